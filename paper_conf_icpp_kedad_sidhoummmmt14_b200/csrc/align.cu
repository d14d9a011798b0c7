// Best local alignment of selected (query, DB sequence) pairs on sm_100a
// (SURVEY 8(f) f1): the end cell of the maximal H, the start cell and the path.
//
// "each element ... keeps the cell that was used to produce
// the value", followed back from the cell of the maximal score.  Tie-breaks
// (reading R-13, the oracle's): end cell = maximal H with the
// smallest column j, then the smallest row i; at an H cell the diagonal is
// preferred, then E, then F; inside a gap, opening is preferred to extending.
//
// Two launches per batch of pairs:
//   align_fwd_kernel  one CTA per pair (persistent, items from a counter), the
//                     chained-warp wavefront of the long-pair mode in int32:
//                     lane k of a warp owns ALIGN_R = 8 rows of a 256-row
//                     strip and at step t computes column t - k; strips go
//                     round-robin to the 8 warps, each consuming the strip
//                     above through a link row + shared progress counter.
//                     Every cell emits a 4-bit traceback code; the 8 codes of
//                     a lane form one u32 word, stored at [strip][t][lane] so
//                     that the 32 lanes of a step write 128 contiguous bytes.
//   align_tb_kernel   one thread per pair walks the codes from the end cell
//                     (dependent loads, O(m + n) steps) and emits run-length
//                     operations, then flips them into start-to-end order.
//
// Traceback code of cell (i, j) (values as in the oracle: E and F here are the
// relu-clamped values of the scoring kernels; a code is consulted only on the
// path, where E, F > 0, so clamping never changes a decision):
//   bits 0-1  H source: 0 = H == 0 (stop), 1 = H == H_{i-1,j-1} + S_ij,
//             2 = H == E_ij, 3 = otherwise (F_ij)
//   bit 2     E_ij == H_{i,j-1} - Gs - Ge   (gap opened here, Eq. (3))
//   bit 3     F_ij == H_{i-1,j} - Gs - Ge   (gap opened here, Eq. (4))
#include <algorithm>

#include "sw_internal.h"
#include "sw_device.cuh"

namespace swdual {

namespace {
constexpr int8_t PAD_S = -64;  // S[.][PAD] = S[PAD][.] (reading R-12)
constexpr int ALIGN_LAG = 16;

struct Best {
  int v, j, i;  // value, 1-based column, 1-based row
};
__device__ __forceinline__ bool better(const Best& a, const Best& b) {
  return a.v > b.v || (a.v == b.v && (a.j < b.j || (a.j == b.j && a.i < b.i)));
}
}  // namespace

// TW = warps per pair ("team"): 8 chains the strips of tall queries across the
// CTA; 1 lets every warp take its own pair (queries of one 256-row strip, where
// a whole CTA per pair would leave 7 warps idle).
template <int TW>
__device__ __forceinline__ void team_sync() {
  if constexpr (TW == 1) __syncwarp();
  else if constexpr (TW == ALIGN_WARPS) __syncthreads();
  else asm volatile("bar.sync %0, %1;" :: "r"(1 + int(threadIdx.x >> 5) / TW), "r"(TW * 32) : "memory");
}

template <int TW>
__global__ void __launch_bounds__(ALIGN_WARPS * 32) align_fwd_kernel(AlignArgs a) {
  constexpr int R = ALIGN_R;
  constexpr int W = TW;  // warps chained on one pair
  constexpr int SW = 33;
  __shared__ int32_t sm[SW * SW];
  __shared__ int s_prog_all[ALIGN_WARPS];
  __shared__ Best s_best_all[ALIGN_WARPS];
  __shared__ int s_item_all[ALIGN_WARPS / TW];
  for (int x = threadIdx.x; x < SW * SW; x += blockDim.x) {
    const int r = x / SW, c = x % SW;
    sm[x] = (r < a.alpha && c < a.alpha) ? int(a.matrix[r * a.alpha + c]) : int(PAD_S);
  }
  const int lane = threadIdx.x & 31, team = (threadIdx.x >> 5) / TW, warp = (threadIdx.x >> 5) % TW;
  const bool lead = lane == 0, tail = lane == 31;
  int* s_prog = s_prog_all + team * TW;
  Best* s_best = s_best_all + team * TW;
  int2* __restrict__ links = a.links + ((size_t)blockIdx.x * ALIGN_WARPS + size_t(team) * TW) * a.bcap;
  const int pad = a.alpha;
  const int nGe = -a.Ge, nGsGe = -(a.Gs + a.Ge);
  const uint2 padw = pad_codes4(pad, a.nib);
  __syncthreads();  // matrix staged
  for (;;) {
    team_sync<TW>();
    if (warp == 0 && lane == 0) s_item_all[team] = atomicAdd(a.work_counter, 1);
    if (warp == 0 && lane < TW) s_prog[lane] = -1;
    team_sync<TW>();
    // TW = 8: sub-item x = (pair, CTA c of K) -- tall pairs are split over K = strips/8
    // CTAs, CTA c taking strips 8c .. 8c+7 (the host sizes K for one round), chained CTA
    // to CTA through global rows + GPU-scope counters like the re-score kernel.
    int item, c = 0, K = 1, sub = 0;
    if constexpr (TW == ALIGN_WARPS) {
      sub = s_item_all[team];
      if (sub >= a.n_sub) break;
      const int2 xm = a.submap[sub];
      item = xm.x;
      c = xm.y;
      K = a.items[item].K;
    } else {
      item = a.item_begin + s_item_all[team];
      if (item >= a.item_begin + a.n_launch) break;
    }
    const int sub0 = sub - c;  // this pair's first sub-item: its global rows / counters / partials
    const AlignItem it = a.items[item];
    const PairRec pr = a.pairs[it.pair];
    const uint8_t* qc = a.qcodes + a.qoff[it.q];
    const int m = int(a.qoff[it.q + 1] - a.qoff[it.q]);
    const int L = (it.n + 3) & ~3;  // this sequence's columns, in whole 4-column words
    const int T = L + 32;           // steps per strip (= trace words per lane per strip)
    const int half = it.half;
    const int nstrips = (m + 32 * R - 1) / (32 * R);

    uint32_t* __restrict__ trace = a.trace + it.trace_off;
    const int jw = W - 1 - warp;  // producers on higher warp ids
    Best acc{0, 0x7fffffff, 0x7fffffff};
    for (int r = 0;; ++r) {
      const int s = W * (K * r + c) + jw;
      if (s >= nstrips || L == 0) break;
      const bool rd = s > 0, wr = s + 1 < nstrips;
      Link lk{};
      const int2* rp;
      int2* wp;
      if (jw > 0 || K == 1) {
        const int jl = (jw + W - 1) % W;
        rp = links + (size_t)jl * a.bcap + 31;
        lk.in = &s_prog[jl];
      } else {  // first warp of a CTA: the strip above is the previous CTA's last
        const int pc = (c + K - 1) % K;
        rp = a.grows + (int64_t)(sub0 + pc) * a.bcap + 31;
        lk.in = a.gflags + sub0 + pc;
        lk.in_gpu = true;
      }
      lk.in_base = (s - 1) << 20;
      if (jw < W - 1 || K == 1) {
        wp = links + (size_t)jw * a.bcap;
        lk.out = &s_prog[jw];
      } else {
        wp = a.grows + (int64_t)(sub0 + c) * a.bcap;
        lk.out = a.gflags + sub0 + c;
        lk.out_gpu = true;
      }
      lk.out_base = s << 20;
      int qr[R], Hl[R], E[R];
#pragma unroll
      for (int rr = 0; rr < R; ++rr) {
        const int row = s * 32 * R + lane * R + rr;
        qr[rr] = (row < m ? int(qc[row]) : pad) * SW;
        Hl[rr] = 0;
        E[rr] = 0;
      }
      const int row0 = s * 32 * R + lane * R + 1;  // 1-based row of rr = 0
      uint32_t* __restrict__ tw = trace + (int64_t)s * T * 32 + lane;
      int hdiag = 0, sH = 0, sF = 0, sC = pad;
      uint32_t eob = 0;  // bit rr: E of this column's row rr was opened (from H of the previous column)
      const int2 z2 = make_int2(0, 0);
      uint2 cw = padw;
      int2 tb0 = z2, tb1 = z2, tb2 = z2, tb3 = z2;
      int seen = -1;
      Best sb{0, 0x7fffffff, 0x7fffffff};  // this strip's best of this lane (first hit in (j, i) order)
      if (rd) wait_progress(lk, lk.in_base + min(4 + 31 + ALIGN_LAG, L + 32), seen);
      if (lead) {
        cw = load_codes4(a.stream, pr.off, 0, a.nib);
        if (rd) { tb0 = __ldcg(rp + 0); tb1 = __ldcg(rp + 1); tb2 = __ldcg(rp + 2); tb3 = __ldcg(rp + 3); }
      }
      __syncwarp();
      for (int t0 = 0; t0 < T; t0 += 4) {
        const uint2 cwc = cw;
        const int2 c0 = tb0, c1 = tb1, c2 = tb2, c3 = tb3;
        if (rd && t0 + 4 < L) wait_progress(lk, lk.in_base + min(t0 + 8 + 31 + ALIGN_LAG, L + 32), seen);
        if (lead) {
          if (t0 + 4 < L) {
            cw = load_codes4(a.stream, pr.off, t0 + 4, a.nib);
            if (rd) {
              tb0 = __ldcg(rp + t0 + 4); tb1 = __ldcg(rp + t0 + 5); tb2 = __ldcg(rp + t0 + 6); tb3 = __ldcg(rp + t0 + 7);
            }
          } else {
            cw = padw;
            tb0 = z2; tb1 = z2; tb2 = z2; tb3 = z2;
          }
        }
        __syncwarp();
#pragma unroll
        for (int jj = 0; jj < 4; ++jj) {
          int rH = __shfl_up_sync(FULL, sH, 1);
          int rF = __shfl_up_sync(FULL, sF, 1);
          int rC = __shfl_up_sync(FULL, sC, 1);
          if (lead) {
            rC = code_of(cwc, jj, half, a.nib);
            const int2 tv = (jj == 0) ? c0 : (jj == 1) ? c1 : (jj == 2) ? c2 : c3;
            rH = tv.x;
            rF = tv.y;
          }
          // beyond this sequence's end the lane sees PAD columns (and so does lane 0 of
          // the strip below through the link row); they never win the end cell
          const int col = t0 + jj - lane + 1;  // 1-based column of this step
          int hd = hdiag;
          hdiag = rH;
          int F = rF;
          // F_{i,j} of row 0 opened from H_{i-1,j} (the row above): decided where F was formed
          uint32_t fo = (F == rH + nGsGe) ? 8u : 0u;
          uint32_t word = 0, eon = 0;
#pragma unroll
          for (int rr = 0; rr < R; ++rr) {
            const int dg = hd + sm[qr[rr] + rC];
            const int e = E[rr];
            const int h = max(max(dg, e), F);                         // Eq. (2) (E, F >= 0)
            const uint32_t src = h == 0 ? 0u : h == dg ? 1u : h == e ? 2u : 3u;
            word |= (src | ((eob >> rr) & 1u) * 4u | fo) << (4 * rr);
            if (h > sb.v) { sb.v = h; sb.j = col; sb.i = row0 + rr; }
            hd = Hl[rr];
            Hl[rr] = h;
            const int tt = h + nGsGe;
            const int ex = e + nGe, fx = F + nGe;
            eon |= (tt >= ex ? 1u : 0u) << rr;                        // E_{i,j+1}: open wins ties
            fo = tt >= fx ? 8u : 0u;                                  // F_{i+1,j}: open wins ties
            E[rr] = max(max(ex, tt), 0);                              // Eq. (3), next column
            F = max(max(fx, tt), 0);                                  // Eq. (4), next row
          }
          eob = eon;
          tw[(int64_t)(t0 + jj) * 32] = word;
          sH = Hl[R - 1];
          sF = F;
          sC = rC;
          if (wr && tail) __stcg(wp + t0 + jj, make_int2(sH, sF));
        }
        if (wr && tail) {
          if (!lk.out_gpu) st_release_cta(lk.out, lk.out_base + t0 + 4);
          else if (((t0 >> 2) & 3) == 3 || t0 + 4 >= T) st_release_gpu(lk.out, lk.out_base + t0 + 4);
        }
      }
      if (better(sb, acc)) acc = sb;
    }
    // CTA-wide lexicographic maximum (value desc, column asc, row asc)
#pragma unroll
    for (int off = 16; off > 0; off >>= 1) {
      Best o;
      o.v = __shfl_xor_sync(FULL, acc.v, off);
      o.j = __shfl_xor_sync(FULL, acc.j, off);
      o.i = __shfl_xor_sync(FULL, acc.i, off);
      if (better(o, acc)) acc = o;
    }
    if (lane == 0) s_best[warp] = acc;
    team_sync<TW>();
    if (warp == 0 && lane == 0) {
      Best b = s_best[0];
      for (int w = 1; w < W; ++w)
        if (better(s_best[w], b)) b = s_best[w];
      if (K == 1) {
        a.best[item] = b.v > 0 ? make_int4(b.v, b.i, b.j, 0) : make_int4(0, 0, 0, 0);
      } else {  // the last of the K CTAs merges their maxima in the same order
        a.partial[sub0 + c] = make_int4(b.v, b.j, b.i, 0);
        __threadfence();
        if (atomicAdd(a.done + item, 1) == K - 1) {
          __threadfence();
          Best m{0, 0x7fffffff, 0x7fffffff};
          for (int x = 0; x < K; ++x) {
            const int4 p = __ldcg(a.partial + sub0 + x);
            const Best o{p.x, p.y, p.z};
            if (better(o, m)) m = o;
          }
          a.best[item] = m.v > 0 ? make_int4(m.v, m.i, m.j, 0) : make_int4(0, 0, 0, 0);
        }
      }
    }
  }
}

// Traceback of one item per thread, in the oracle's order.
__global__ void align_tb_kernel(AlignArgs a) {
  const int item = blockIdx.x * blockDim.x + threadIdx.x;
  if (item >= a.n_items) return;
  const AlignItem it = a.items[item];
  const int4 b = a.best[item];
  int32_t* out = a.out + (int64_t)item * 6;
  if (b.x <= 0) {
    out[0] = 0; out[1] = out[2] = out[3] = out[4] = -1; out[5] = 0;
    return;
  }
  const int T = ((it.n + 3) & ~3) + 32;
  const uint32_t* __restrict__ trace = a.trace + it.trace_off;
  uint32_t* __restrict__ ops = a.ops + it.ops_off;
  auto code = [&](int i, int j) -> uint32_t {  // 1-based cell
    const int r = i - 1, c = j - 1;
    const int s = r >> 8, ln = (r >> 3) & 31, rr = r & 7;
    const uint32_t w = __ldcg(trace + ((int64_t)s * T + c + ln) * 32 + ln);
    return (w >> (4 * rr)) & 15u;
  };
  int i = b.y, j = b.z, state = 0, n = 0;
  int run_op = -1, run_len = 0;
  bool overflow = false;
  for (;;) {
    int op;
    if (state == 0) {
      if (i == 0 || j == 0) break;
      const uint32_t c = code(i, j) & 3u;
      if (c == 0) break;
      if (c == 1) { op = 0; --i; --j; }
      else { state = int(c) - 1; continue; }  // 2 -> E (1), 3 -> F (2)
    } else if (state == 1) {
      op = 2;
      state = (code(i, j) & 4u) ? 0 : 1;
      --j;
    } else {
      op = 1;
      state = (code(i, j) & 8u) ? 0 : 2;
      --i;
    }
    if (op == run_op) ++run_len;
    else {
      if (run_len) {
        if (n < it.ops_cap) ops[n] = (uint32_t(run_len) << 2) | uint32_t(run_op);
        else overflow = true;
        ++n;
      }
      run_op = op;
      run_len = 1;
    }
  }
  if (run_len) {
    if (n < it.ops_cap) ops[n] = (uint32_t(run_len) << 2) | uint32_t(run_op);
    else overflow = true;
    ++n;
  }
  if (!overflow)
    for (int k = 0; k < n / 2; ++k) {
      const uint32_t x = ops[k];
      ops[k] = ops[n - 1 - k];
      ops[n - 1 - k] = x;
    }
  out[0] = b.x;
  out[1] = i;        // 0-based first query residue (the walk stops on the cell before it)
  out[2] = b.y - 1;  // 0-based last query residue
  out[3] = j;
  out[4] = b.z - 1;
  out[5] = overflow ? -n : n;
}

// items [0, n_single) have one strip (warp per pair), [n_single, n_items) are
// taller (CTA per pair); counters[0..1] zeroed by the caller.
cudaError_t launch_align(int grid, int n_single, const AlignArgs& a0, int* counters, cudaStream_t st) {
  if (a0.n_items <= 0) return cudaSuccess;
  AlignArgs a = a0;
  if (n_single > 0) {
    a.item_begin = 0;
    a.n_launch = n_single;
    a.work_counter = counters;
    const int g = std::max(1, std::min(grid, (n_single + ALIGN_WARPS - 1) / ALIGN_WARPS));
    align_fwd_kernel<1><<<g, ALIGN_WARPS * 32, 0, st>>>(a);
    cudaError_t e = cudaGetLastError();
    if (e != cudaSuccess) return e;
  }
  if (a0.n_sub > 0) {
    a.work_counter = counters + 1;
    align_fwd_kernel<ALIGN_WARPS><<<std::min(grid, a0.n_sub), ALIGN_WARPS * 32, 0, st>>>(a);
    cudaError_t e = cudaGetLastError();
    if (e != cudaSuccess) return e;
  }
  align_tb_kernel<<<(a0.n_items + 127) / 128, 128, 0, st>>>(a0);
  return cudaGetLastError();
}

}  // namespace swdual
