// SWDUAL hot-path kernels for sm_100a: query-profile builds, the inter-task
// s16x2 DPX scoring kernels (short pairs), the intra-task chained-warp kernel
// (long pairs), the exact int32 re-score, the mapped-output zeroing and the
// gathered-block merge.
//
// Inter-task kernels (the paper's "very coarse-grained" split
// across workers, with the "fine-grained" wavefront inside a
// worker, L202-216 / Fig. 2):
//   * a lane GROUP of G lanes scores one database pair (two length-neighbours,
//     one per s16x2 half) against one query (mode 0), or one database sequence
//     against a query PAIR (mode 1, two queries per s16x2 register);
//   * lane k of the group owns R consecutive query rows of the current strip
//     (strip height G*R rows); at step t it computes column t-k, so the group
//     sweeps the matrix as an anti-diagonal wave: the bottom row (H, F) and the
//     residue codes travel one lane down per step over warp shuffles;
//   * queries taller than one strip are done in passes; the last lane writes the
//     strip's bottom row to a per-group global boundary row that lane 0 reads
//     in the next pass;
//   * the query profile of the current strip sits in shared memory;
//   * CTAs are persistent and take chunks of NT/G pairs from an atomic counter,
//     pairs sorted longest first.
// Each mode is its own kernel (its own register budget: the query-pair kernel
// holds 2 CTAs per SM at 128 registers with R up to 32).
#include <algorithm>
#include <cstdio>
#include "sw_internal.h"
#include "sw_device.cuh"

namespace swdual {

constexpr int8_t PAD_SCORE = -64;  // S[.][PAD] = S[PAD][.] <= 0 (reading R-12)
// Intra-task mode: a strip starts consuming the row above only once its
// producer is this many columns ahead, so producer and consumer warps of a
// chain run decoupled instead of in lock-step (the consumer then rarely waits).
constexpr int LINK_LAG = 32;
constexpr int RESCORE_LAG = 16;  // re-score chains: one round per CTA, short lag keeps the critical path short

// ---------------------------------------------------------------------------
// Query profile: prof[s][a][k][r] = S[q[s*G*R + k*R + r]][a]  (int8)
//   a < alpha: matrix column a; a == alpha: PAD; rows >= m: PAD.
__global__ void build_profile_kernel(const uint8_t* __restrict__ q, int m, const int8_t* __restrict__ M,
                                     int alpha, ProfGeom g, uint8_t* __restrict__ prof) {
  const int64_t total = (int64_t)g.n_strips * g.SB;
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < total;
       i += (int64_t)gridDim.x * blockDim.x) {
    const int s = int(i / g.SB);
    const int rem = int(i - (int64_t)s * g.SB);
    int8_t v = 0;
    if (rem < g.NL * g.LS) {
      const int a = rem / g.LS;
      const int rr = rem - a * g.LS;
      int k, r;
      if (g.il) {  // [unit u][lane k][UB bytes]
        const int u = rr / (g.G * g.UB);
        const int w = rr - u * (g.G * g.UB);
        k = w / g.UB;
        r = u * g.UB + (w - k * g.UB);
      } else {     // [lane k][LB bytes] (LS may be padded past G lanes)
        k = rr / g.LB;
        r = rr - k * g.LB;
      }
      if (k < g.G && r < g.R) {
        const int row = s * g.G * g.R + k * g.R + r;
        v = (row < m && a < alpha) ? M[q[row] * alpha + a] : PAD_SCORE;
      }
    }
    prof[i] = uint8_t(v);
  }
}

cudaError_t launch_build_profile(const uint8_t* q, int m, const int8_t* matrix, int alpha, const ProfGeom& g,
                                 uint8_t* prof, cudaStream_t st) {
  const int64_t total = (int64_t)g.n_strips * g.SB;
  int grid = int((total + 255) / 256);
  if (grid > 4096) grid = 4096;
  if (grid < 1) grid = 1;
  build_profile_kernel<<<grid, 256, 0, st>>>(q, m, matrix, alpha, g, prof);
  return cudaGetLastError();
}

// Query-pair profile: 32-bit word per (strip, letter, lane, row):
//   low 16 = S[qa[row]][a], high 16 = S[qb[row]][a]  (PAD rows / letters: PAD_SCORE)
__global__ void build_profile_q2_kernel(const uint8_t* __restrict__ qa, int ma, const uint8_t* __restrict__ qb,
                                        int mb, const int8_t* __restrict__ M, int alpha, int G, int R, int LB2,
                                        int LS2, int n_strips, int SB2, uint32_t* __restrict__ prof) {
  const int64_t total = (int64_t)n_strips * (SB2 / 4);
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < total;
       i += (int64_t)gridDim.x * blockDim.x) {
    const int s = int(i / (SB2 / 4));
    const int rem = int(i - (int64_t)s * (SB2 / 4)) * 4;  // byte offset within the strip
    uint32_t v = 0;
    if (rem < (alpha + 1) * LS2) {
      const int a = rem / LS2;
      const int rr = rem - a * LS2;
      const int k = rr / LB2;
      const int r = (rr - k * LB2) / 4;
      if (k < G && r < R) {
        const int row = s * G * R + k * R + r;
        // rows past a query, and PAD codes (= alpha) that pad packed queries to whole strips
        const int ca = row < ma ? qa[row] : alpha, cb = row < mb ? qb[row] : alpha;
        const int va = (ca < alpha && a < alpha) ? M[ca * alpha + a] : PAD_SCORE;
        const int vb = (cb < alpha && a < alpha) ? M[cb * alpha + a] : PAD_SCORE;
        v = (uint32_t(va) & 0xffffu) | (uint32_t(vb) << 16);
      }
    }
    prof[i] = v;
  }
}

cudaError_t launch_build_profile_q2(const uint8_t* qa, int ma, const uint8_t* qb, int mb, const int8_t* matrix,
                                    int alpha, int G, int R, int LB2, int LS2, int n_strips, int SB2, uint8_t* prof,
                                    cudaStream_t st) {
  const int64_t total = (int64_t)n_strips * (SB2 / 4);
  int grid = int((total + 255) / 256);
  if (grid > 4096) grid = 4096;
  if (grid < 1) grid = 1;
  build_profile_q2_kernel<<<grid, 256, 0, st>>>(qa, ma, qb, mb, matrix, alpha, G, R, LB2, LS2, n_strips, SB2,
                                                reinterpret_cast<uint32_t*>(prof));
  return cudaGetLastError();
}

// ---------------------------------------------------------------------------
__device__ __forceinline__ void copy_strip(uint8_t* dst, const uint8_t* __restrict__ src, int bytes) {
  const uint4* s = reinterpret_cast<const uint4*>(src);
  if ((reinterpret_cast<uintptr_t>(dst) & 15) == 0) {
    uint4* d = reinterpret_cast<uint4*>(dst);
    for (int i = threadIdx.x; i < bytes / 16; i += blockDim.x) d[i] = __ldg(s + i);
  } else {  // bank-skewed copy (4-byte aligned)
    uint32_t* d = reinterpret_cast<uint32_t*>(dst);
    for (int i = threadIdx.x; i < bytes / 16; i += blockDim.x) {
      const uint4 v = __ldg(s + i);
      d[4 * i] = v.x; d[4 * i + 1] = v.y; d[4 * i + 2] = v.z; d[4 * i + 3] = v.w;
    }
  }
}
// byte offset of bank-spread copy cp of the short strip profile
__device__ __forceinline__ int copy_off(int cp, int csx, uint32_t skew) {
  return cp * csx + 4 * int((skew >> (8 * cp)) & 0xffu);
}

template <int R>
struct SubLanes {
  // Each lane runs V "sub-lanes" of R/V rows, the second one column behind the
  // first: two independent dependency chains per step (twice the ILP of the
  // row-to-row F chain), at the cost of a (V*G - 1)-column wave fill.
  static constexpr int V = (R % 8 == 0) ? 2 : 1;
};

// Boundary cells of a strip pass.  Short items: a per-group row in global memory
// (written in one pass, read in the next).  Long items: a shared-memory ring
// between two concurrently running warps (producer progress / consumer progress
// counters, LONG_RING steps of slack) or, for the round wrap, a global row.
struct Chain {
  bool in_ring, out_ring;    // rings (shared memory) or global rows
  uint32_t in_sring, out_sring;  // shared-window addresses of the rings
  int* in_prog;              // producer progress (steps written, monotone across rounds), shared
  int* in_cons;              // this warp's consumption of its input, published for the producer
  int* out_prog;             // this warp's output progress
  const int* out_cons;       // consumption of this warp's output by its consumer
  int in_base, out_base;     // step index (monotone across rounds) of the producer's / this warp's step 0
  const uint2* grow_in;      // global input row (round wrap)
  uint2* grow_out;           // global output row (round wrap)
};

__device__ __forceinline__ uint4 lds128v(uint32_t a) { return lds128(a); }
__device__ __forceinline__ void sts64(uint32_t a, uint2 v) {
  asm volatile("st.shared.v2.u32 [%0], {%1, %2};" :: "r"(a), "r"(v.x), "r"(v.y) : "memory");
}

// Warp-uniform spin until *p >= need: lane `who` (the lane whose later shared
// memory accesses the counter orders) polls with acquire, the value is broadcast.
__device__ __forceinline__ void wait_geq(const int* p, int need, int& seen, int who) {
  if (seen >= need) return;
  for (;;) {
    int v = 0;
    if ((threadIdx.x & 31) == who) v = ld_acquire_cta(p);
    v = __shfl_sync(FULL, v, who);
    if (v >= need) { seen = v; return; }
    __nanosleep(32);
  }
}

// One strip pass of a lane group over one pair: G lanes x R rows, columns
// streamed as an anti-diagonal wave.  Boundary rows: lane 0 reads the strip
// above at rp[c] (c = column, rp = row base + G - 1), lane G-1 writes this
// strip's bottom row at wp[t] (t = step).  LINKED (long items, G = 32): the
// row above is produced concurrently by another warp of the CTA (Chain).
// NIB: the pair's columns are bytes of two 4-bit codes (nucleotide DBs, SURVEY 8(f)
// f4): lane 0 loads 4 columns per 32-bit word and spreads each byte into the
// 16-bit pair word (two 8-bit codes) the rest of the pass uses.
template <int G, int R, bool LINKED, bool Q2 = false, int US = (Q2 ? 16 : ((R % 8 == 0) ? 8 : 4)), bool NIB = false>
__device__ __forceinline__ void strip_pass(const uint8_t* sprof, int LS, int LB, const void* pstream, int L,
                                           int T, int k, bool rd, bool wr, const uint2* __restrict__ rp,
                                           uint2* __restrict__ wp, const Chain& ch, uint32_t code_pad2,
                                           uint32_t nGe, uint32_t nGsGe, uint32_t& best, uint32_t shift = 0) {
  constexpr int V = SubLanes<R>::V;
  constexpr int VG = V * G;   // width of the wave in sub-lanes
  constexpr int RH = R / V;   // rows per sub-lane
  // code-ahead pipeline (below): single-query short items only -- measured C2 +3 %; the
  // query-pair kernel (C3) loses 1 % to the extra registers, 32-lane groups gain nothing
  constexpr bool CA = !Q2 && G < 32;
  uint32_t HA[R], E[R];
#pragma unroll
  for (int r = 0; r < R; ++r) { HA[r] = 0; E[r] = 0; }
  const uint32_t sbase = static_cast<uint32_t>(__cvta_generic_to_shared(sprof));
  uint32_t hdiag = 0, sH = 0, sF = 0, sC = code_pad2;
  const uint2* __restrict__ codes = reinterpret_cast<const uint2*>(pstream);
  const uint32_t* __restrict__ codes4 = reinterpret_cast<const uint32_t*>(pstream);
  const uint32_t pad4 = NIB ? ((code_pad2 & 0xfu) | ((code_pad2 >> 4) & 0xf0u)) * 0x01010101u
                            : code_pad2 | (code_pad2 << 16);
  const uint32_t laneoff = uint32_t(k) * LB;
  const bool lead = (k == 0), tail = (k == G - 1);
  const uint2 z2 = make_uint2(0, 0);
  // second sub-lane: its inputs are the first sub-lane's outputs of the previous step
  uint32_t hdiag1 = 0, cH = 0, cF = 0, pC = code_pad2;
  const uint32_t pad_row = sbase + (code_pad2 & 0xffu) * LS + laneoff;
  uint32_t ppa = pad_row, ppb = pad_row;
  // input index of sub-lane 0 of lane 0 for column c: c + VG - 1 (producer step)
  const int ioff = VG - 1;
  int seen_in = -1, seen_out = -1;

  // lane 0 prefetch of block 0: 4 columns of codes and (if rd) 4 boundary cells.
  // L and t0 are multiples of 4, so one compare guards a whole block.
  auto load_codes = [&](int t0) -> uint2 {
    if constexpr (NIB) return make_uint2(__ldcs(codes4 + (t0 >> 2)), 0u);
    else return __ldcs(codes + (t0 >> 2));
  };
  auto load_block = [&](int t0, uint2& cw, uint2& b0, uint2& b1, uint2& b2, uint2& b3) {
    if (!CA) cw = load_codes(t0);
    if (rd) {
      if constexpr (LINKED) {
        if (ch.in_ring) {
          const int x = ch.in_base + t0 + ioff;  // 3 mod 4 (ioff = 63): the 4 cells one by one
          const uint32_t a0 = ch.in_sring + uint32_t((x & (LONG_RING - 1)) * 8);
          const uint32_t a1 = ch.in_sring + uint32_t(((x + 1) & (LONG_RING - 1)) * 8);
          const uint32_t a2 = ch.in_sring + uint32_t(((x + 2) & (LONG_RING - 1)) * 8);
          const uint32_t a3 = ch.in_sring + uint32_t(((x + 3) & (LONG_RING - 1)) * 8);
          b0 = lds64(a0); b1 = lds64(a1); b2 = lds64(a2); b3 = lds64(a3);
        } else {
          const uint2* g = ch.grow_in + t0 + ioff;
          b0 = __ldcg(g); b1 = __ldcg(g + 1); b2 = __ldcg(g + 2); b3 = __ldcg(g + 3);
        }
      } else {  // rp is 32-byte aligned at rp + ioff (see the bb base in short_body)
        const uint4 x = *reinterpret_cast<const uint4*>(rp + t0 + ioff);
        const uint4 y = *reinterpret_cast<const uint4*>(rp + t0 + ioff + 2);
        b0 = make_uint2(x.x, x.y); b1 = make_uint2(x.z, x.w); b2 = make_uint2(y.x, y.y); b3 = make_uint2(y.z, y.w);
      }
    }
  };
  // long items: progress this warp's consumer needs before block t0's prefetch
  auto wait_in = [&](int t0) {
    if constexpr (LINKED) {
      if (rd) wait_geq(ch.in_prog, ch.in_base + min(t0 + 4 + ioff + LINK_LAG, L + VG), seen_in, 0);
    }
  };
  uint2 cw = make_uint2(pad4, pad4);
  uint2 tb0 = z2, tb1 = z2, tb2 = z2, tb3 = z2;
  // code of column jj (0..3) of a 4-column block word: the 16-bit pair word (two 8-bit codes)
  auto code_at = [&](uint2 w, int jj) -> uint32_t {
    if constexpr (NIB) {
      const uint32_t b8 = (w.x >> (8 * jj)) & 0xffu;
      return (b8 & 0xfu) | ((b8 & 0xf0u) << 4);
    } else {
      const uint32_t x = (jj < 2) ? w.x : w.y;
      return (jj & 1) ? (x >> 16) : (x & 0xffffu);
    }
  };
  // Code-ahead pipeline: the code a lane uses at step t is its upper neighbour's code of
  // step t - V, known a step early, so it is shuffled one step ahead (nC) and the
  // profile address of the next step is off the shuffle -> LDS path.  The lead lane
  // reads its codes two blocks ahead (cwn: the next block).
  uint2 cwn = make_uint2(pad4, pad4);
  if (L > 0) {
    wait_in(0);
    if (lead) {
      load_block(0, cw, tb0, tb1, tb2, tb3);
      if (CA) {
        cw = load_codes(0);
        if (4 < L) cwn = load_codes(4);
      }
    }
  }
  uint32_t nC = lead ? code_at(cw, 0) : code_pad2;
  __syncwarp();
  for (int t0 = 0; t0 < T; t0 += 4) {
    const uint2 cwc = cw;
    const uint2 cwnc = cwn;
    const uint2 c0 = tb0, c1 = tb1, c2 = tb2, c3 = tb3;
    if (t0 + 4 < L) wait_in(t0 + 4);
    if constexpr (LINKED) {
      // ring space for this block's outputs (the consumer may lag by up to LONG_RING steps)
      if (wr && ch.out_ring) wait_geq(ch.out_cons, ch.out_base + t0 + 4 - LONG_RING, seen_out, G - 1);
    }
    if (lead) {
      if (t0 + 4 < L) {
        load_block(t0 + 4, cw, tb0, tb1, tb2, tb3);
      } else {
        cw = make_uint2(pad4, pad4);
        tb0 = z2; tb1 = z2; tb2 = z2; tb3 = z2;
      }
      if (CA) {
        cw = cwnc;
        cwn = (t0 + 8 < L) ? load_codes(t0 + 8) : make_uint2(pad4, pad4);
      }
    }
    __syncwarp();
#pragma unroll
    for (int j = 0; j < 4; ++j) {
      uint32_t rH = __shfl_up_sync(FULL, sH, 1, G);
      uint32_t rF = __shfl_up_sync(FULL, sF, 1, G);
      uint32_t rC;
      if (CA) {
        rC = nC;
        uint32_t xC = __shfl_up_sync(FULL, V == 2 ? pC : rC, 1, G);  // this lane's code of the next step
        if (lead) xC = (j < 3) ? code_at(cwc, j + 1) : code_at(cwnc, 0);
        nC = xC;
      } else {
        rC = __shfl_up_sync(FULL, sC, 1, G);
        if (lead) rC = code_at(cwc, j);
      }
      if (lead) {
        const uint2 tv = (j == 0) ? c0 : (j == 1) ? c1 : (j == 2) ? c2 : c3;
        rH = tv.x;
        rF = tv.y;
      }
      uint32_t pa, pb;
      if constexpr (Q2) {  // one DB sequence (byte `shift` of the pair word) against two queries
        pa = sbase + ((rC >> shift) & 0xffu) * LS + laneoff;
        pb = pa;
      } else {
        pa = sbase + (rC & 0xffu) * LS + laneoff;
        pb = sbase + (rC >> 8) * LS + laneoff;
      }
      if constexpr (V == 2) {
        uint32_t h1 = cH, f1 = cF;
        if constexpr (Q2) {  // measured: +3% for the query-pair mode, -2% with the PRMT (mode 0)
          gotoh_rows_dual<R, Q2, US>(HA, E, best, hdiag, pa, pb, rH, rF, hdiag1, ppa, ppb, h1, f1, nGe, nGsGe);
        } else {
          // sub-lane 1 (rows RH..R-1, column t-1) first: it reads rows it owns only
          gotoh_rows_inplace<R, RH, R, Q2, US>(HA, E, best, hdiag1, ppa, ppb, h1, f1, nGe, nGsGe);
          gotoh_rows_inplace<R, 0, RH, Q2, US>(HA, E, best, hdiag, pa, pb, rH, rF, nGe, nGsGe);
        }
        cH = rH;
        cF = rF;
        ppa = pa;
        ppb = pb;
        sH = h1;
        sF = f1;
        sC = pC;
        pC = rC;
      } else {
        gotoh_rows_inplace<R, 0, R, Q2, US>(HA, E, best, hdiag, pa, pb, rH, rF, nGe, nGsGe);
        sH = rH;
        sF = rF;
        sC = rC;
      }
      if (wr && tail) {
        if constexpr (LINKED) {
          if (ch.out_ring) sts64(ch.out_sring + uint32_t(((ch.out_base + t0 + j) & (LONG_RING - 1)) * 8), make_uint2(sH, sF));
          else __stcg(ch.grow_out + t0 + j, make_uint2(sH, sF));
        } else {
          wp[t0 + j] = make_uint2(sH, sF);
        }
      }
    }
    if constexpr (LINKED) {
      // progress, every 8 columns: release orders this lane's ring writes before the counter
      if (wr && tail && (((t0 >> 2) & 1) || t0 + 4 >= T)) st_release_cta(ch.out_prog, ch.out_base + t0 + 4);
      // consumption: block t0's ring cells were used above (their loads completed), so a
      // relaxed store suffices -- the producer only overwrites cells below this index
      if (rd && ch.in_ring && lead && (((t0 >> 2) & 1) || t0 + 4 >= T))
        st_relaxed_cta(ch.in_cons, ch.in_base + min(t0 + 4 + ioff, T));
    }
  }
  if constexpr (LINKED) {
    if (rd && ch.in_ring && lead) st_relaxed_cta(ch.in_cons, ch.in_base + T);  // everything consumed
  }
}

__device__ __forceinline__ void flag_overflow(int* ovf_count, OvfRec* ovf, int cap, int q, int p, int half) {
  const int e = atomicAdd(ovf_count, 1);
  if (e < cap) ovf[e] = OvfRec{q, p, half, 0};
}

// ---------------------------------------------------------------------------
// Short-pair items: the host ordered all (slot, chunk) items of
// the launch by critical path (strips x pair length), longest first.
// Query-pair strip profiles are staged by the TMA engine: two shared-memory
// buffers, each holding the bank-spread copies of one strip; while the lane groups
// sweep strip s from one buffer, cp.async.bulk fills the other with strip s+1
// (completion counted on that buffer's mbarrier).  One CTA barrier per pass.
struct ProfStage {
  int tag[2];        // (slot << 16 | strip) held / in flight per buffer, -1: none (CTA-uniform)
  uint32_t parity;   // bit b: mbarrier phase parity the next wait on buffer b expects
  uint32_t pending;  // bit b: a bulk copy into buffer b not yet waited for
  uint64_t* mbar;    // [2] in shared memory
};

__device__ __forceinline__ void stage_issue(ProfStage& ps, int b, int tag, const ShortArgs& a, uint8_t* buf,
                                            const uint8_t* src) {
  if (threadIdx.x == 0) {
    fence_proxy_async_smem();  // the buffer's previous strip was read through the generic proxy
    mbar_arrive_expect_tx(ps.mbar + b, uint32_t(a.ncopy * a.SB));
    for (int cp = 0; cp < a.ncopy; ++cp) bulk_g2s(buf + cp * a.cstride, src, uint32_t(a.SB), ps.mbar + b);
  }
  ps.tag[b] = tag;
  ps.pending |= 1u << b;
}

// CG: the gap penalties are the compile-time pair Gs = 10, Ge = 2 (BASELINE's
// configuration): the cell update then encodes -Ge and -(Gs+Ge) as immediates,
// one register operand fewer per VIADDMNMX / VIADD (register-file bandwidth).
template <int G, int R, int NT, bool Q2, bool CG = false, bool NIB = false>
__device__ __forceinline__ void short_item(const ShortArgs& a, int item, uint8_t* smem, int& loaded, ProfStage& ps) {
  const uint32_t nGe = CG ? 0xfffefffeu : a.nGe, nGsGe = CG ? 0xfff4fff4u : a.nGsGe;
  uint8_t* sprof = smem;                         // the strip profile (bank-spread copies)
  constexpr int NG = NT / G;
  const int tid = threadIdx.x;
  const int k = tid & (G - 1);
  const int g = tid / G;
  // per-group boundary row; offset so that &bb[V*G - 1] is 32-byte aligned (bcap % 4 == 0)
  constexpr int BB_PAD = (4 - (G * SubLanes<R>::V - 1) % 4) % 4;
  uint2* __restrict__ bb = a.bbuf + ((size_t)blockIdx.x * NG + g) * (size_t)a.bcap + BB_PAD;
  {
    const int2 sc = a.item_map[item];
    const int sl = sc.x;
    const SlotDesc d = a.slots[sl];
    const int chunk = sc.y;
    int p, half = 0;
    if constexpr (Q2) {  // chunk of NG half-pairs: DB sequence = one half of a pair
      const int hp = chunk * NG + g;
      p = d.pair_begin + (hp >> 1);
      half = hp & 1;
    } else {
      p = d.pair_begin + chunk * NG + g;
    }
    bool valid = p < a.pair_end;
    PairRec pr;
    if (valid) pr = a.pairs[p];
    else { pr.off = 0; pr.len = 0; pr.id0 = -1; pr.id1 = -1; }
    if (Q2 && half && pr.id1 < 0) valid = false;  // odd leftover pair has no high half
    const void* pstream = NIB ? static_cast<const void*>(reinterpret_cast<const uint8_t*>(a.stream) + pr.off)
                              : static_cast<const void*>(a.stream + pr.off);
    int T = pr.len + G * SubLanes<R>::V;          // the last sub-lane finishes column len-1 at step T-2
    if (G < 32) T = __reduce_max_sync(FULL, T);   // warp-uniform trip count (shuffles)
    uint32_t best = 0;
    for (int s = 0; s < d.n_strips; ++s) {
      const int want = (sl << 16) | s;
      const uint8_t* sbuf = sprof;
      if constexpr (Q2) {
        const int bsz = (a.ncopy - 1) * a.cstride + a.SB;
        const int b = s & 1;
        __syncthreads();  // every group is done with strip s-1 (the other buffer) and strip s-2 (this one)
        if (ps.tag[b] != want) stage_issue(ps, b, want, a, sprof + b * ((bsz + 127) & ~127), d.prof + (size_t)s * a.SB);
        if (s + 1 < d.n_strips && ps.tag[b ^ 1] != want + 1)  // prefetch the next strip
          stage_issue(ps, b ^ 1, want + 1, a, sprof + (b ^ 1) * ((bsz + 127) & ~127), d.prof + (size_t)(s + 1) * a.SB);
        if (ps.pending & (1u << b)) {
          mbar_wait(ps.mbar + b, (ps.parity >> b) & 1u);
          ps.parity ^= 1u << b;
          ps.pending &= ~(1u << b);
        }
        sbuf = sprof + b * ((bsz + 127) & ~127);
      } else if (want != loaded) {
        __syncthreads();
        for (int cp = 0; cp < a.ncopy; ++cp)
          copy_strip(sprof + copy_off(cp, a.cstride, a.cskew), d.prof + (size_t)s * a.SB, a.SB);
        __syncthreads();
        loaded = want;
      }
      const uint8_t* gprof = sbuf + copy_off(g & (a.ncopy - 1), a.cstride, a.cskew);  // this group's copy
      if constexpr (Q2) {
        const StripInfo si = d.sinfo[s];
        const bool rd = s > 0 && si.keep != 0;
        if (rd && si.keep != FULL) {  // one half starts a new query: zero its half of the boundary row
          for (int c = k; c < T; c += G) {
            const uint2 v = bb[c];
            bb[c] = make_uint2(v.x & si.keep, v.y & si.keep);
          }
          __syncwarp();
        }
        strip_pass<G, R, false, true, 16, NIB>(gprof, a.LS, a.LB, pstream, pr.len, T, k, rd, s + 1 < d.n_strips,
                                      bb, bb, Chain{}, a.code_pad2, nGe, nGsGe, best, half ? 8u : 0u);
        if (si.emit0 >= 0 || si.emit1 >= 0) {  // a query of either half ends with this strip
          uint32_t bg = best;
#pragma unroll
          for (int o = G / 2; o > 0; o >>= 1) bg = __vmaxs2(bg, __shfl_xor_sync(FULL, bg, o, G));
          if (valid && k == 0) {
            const int id = half ? pr.id1 : pr.id0;
            if (si.emit0 >= 0) {
              const int v = int(int16_t(bg & 0xffffu));
              a.scores_all[(int64_t)si.emit0 * a.n_seqs + id] = v;
              if (v >= a.thr) flag_overflow(a.ovf_count, a.ovf, a.ovf_cap, si.emit0, p, half);
            }
            if (si.emit1 >= 0) {
              const int v = int(int16_t(bg >> 16));
              a.scores_all[(int64_t)si.emit1 * a.n_seqs + id] = v;
              if (v >= a.thr) flag_overflow(a.ovf_count, a.ovf, a.ovf_cap, si.emit1, p, half);
            }
          }
          best &= (si.emit0 >= 0 ? 0xffff0000u : 0xffffffffu) & (si.emit1 >= 0 ? 0x0000ffffu : 0xffffffffu);
        }
      } else {
        strip_pass<G, R, false, false, ((R % 8 == 0) ? 8 : 4), NIB>(gprof, a.LS, a.LB, pstream, pr.len, T, k, s > 0,
                                                                  s + 1 < d.n_strips,
                                bb, bb, Chain{}, a.code_pad2, nGe, nGsGe, best);
      }
    }
    if constexpr (!Q2) {  // mode 0: one query, both halves are DB sequences
#pragma unroll
      for (int o = G / 2; o > 0; o >>= 1) best = __vmaxs2(best, __shfl_xor_sync(FULL, best, o, G));
      if (valid && k == 0) {
        const int lo = int(int16_t(best & 0xffffu)), hi = int(int16_t(best >> 16));
        d.scores0[pr.id0] = lo;
        if (lo >= a.thr) flag_overflow(a.ovf_count, a.ovf, a.ovf_cap, d.qidx0, p, 0);
        if (pr.id1 >= 0) {
          d.scores0[pr.id1] = hi;
          if (hi >= a.thr) flag_overflow(a.ovf_count, a.ovf, a.ovf_cap, d.qidx0, p, 1);
        }
      }
    }
  }
}

// Long-pair items (intra-task mode; the paper's fine-grained
// wavefront across PEs, Fig. 2): one CTA item = one (query, long pair);
// its LONG_W warps run the strips of 32 lanes x LONG_R rows round-robin (round r:
// warp w takes strip LONG_W*r + (LONG_W-1-w); upstream strips on the HIGHER warp
// ids, which the SMSP arbiter favours, so producers keep their lead).  Strip s
// consumes strip s-1's bottom row: inside a round through a shared-memory ring
// (LONG_RING steps; producer progress and consumer progress counters give
// back-pressure), across the round wrap (the last warp's strip -> the first
// warp's strip of the next round, which starts only after the first warp's
// current strip ends) through a global row per CTA.  A pair never spans CTAs:
// every wait is on a warp of the same CTA, so nothing depends on co-residency.
struct LongShared {
  int prog[LONG_W];
  int cons[LONG_W];
  uint32_t best[LONG_W];
};

template <bool NIB, int LR>
__device__ __forceinline__ void long_item(const LongArgs& a, int item, uint8_t* smem, LongShared& sh) {
  constexpr int W = LONG_W;
  // A producer may run LONG_RING - 4 steps ahead of its consumer's last published
  // consumption; the consumer starts only once the producer is ioff + 4 +
  // LINK_LAG steps in, so the ring must hold more than that (else both wait).
  static_assert(LONG_RING - 4 >= (32 * SubLanes<LR>::V - 1) + 4 + LINK_LAG + 16, "ring too short for the lag");
  uint2* rings = reinterpret_cast<uint2*>(smem);                       // [W - 1][LONG_RING]
  uint8_t* lprof = smem + (W - 1) * LONG_RING * sizeof(uint2);         // [W][SBL]
  int* s_prog = sh.prog;
  int* s_cons = sh.cons;
  uint32_t* s_best = sh.best;
  const int tid = threadIdx.x;
  const int lane = tid & 31, warp = tid >> 5;
  {
    if (tid < W) { s_prog[tid] = -1; s_cons[tid] = 0; s_best[tid] = 0; }
    __syncthreads();
    const int2 li = a.lmap[item];  // (query, item within the query), costliest first across queries
    const LongQuery d = a.queries[li.x];
    const int ns = d.n_strips;
    // P pairs per item, GS warps each (host-chosen, P * GS <= W: few idle warp-rounds)
    const int P = d.pack;
    const int GS = d.gs;
    const int grp = warp / GS, wg = warp - grp * GS;
    uint2* wrap = a.wrap + ((size_t)blockIdx.x * a.wrap_groups + (grp < a.wrap_groups ? grp : 0)) * a.wcap;
    const int j = GS - 1 - wg;                   // position of this warp's strip within a round
    const int pidx = li.y * P + grp;
    const bool active = grp < P && pidx < d.n_long;
    PairRec pr;
    if (active) pr = a.pairs[pidx];
    else { pr.off = 0; pr.len = 0; pr.id0 = -1; pr.id1 = -1; }
    constexpr int VG = 32 * SubLanes<LR>::V;
    const int T = pr.len + VG;
    uint32_t best = 0;
    uint8_t* myprof = lprof + warp * a.SBL;
    const int lbase = grp * (GS - 1), cbase = grp * GS;  // this pair's rings and counters
    for (int r = 0; active; ++r) {
      const int s = GS * r + j;  // strip index
      if (s >= ns) break;
      __syncwarp();
      {  // this warp's strip profile -> its own slot
        const uint4* src = reinterpret_cast<const uint4*>(d.prof_long + (size_t)s * a.SBL);
        uint4* dst = reinterpret_cast<uint4*>(myprof);
        for (int i = lane; i < a.SBL / 16; i += 32) dst[i] = __ldg(src + i);
      }
      __syncwarp();
      const bool rd = s > 0, wr = s + 1 < ns;
      Chain ch{};
      ch.out_base = r * T;
      // input: ring j-1 (same round) or the wrap row (previous round, from position GS-1)
      ch.in_ring = j > 0;
      if (j > 0) {
        ch.in_sring = static_cast<uint32_t>(__cvta_generic_to_shared(rings + (size_t)(lbase + j - 1) * LONG_RING));
        ch.in_prog = &s_prog[cbase + j - 1];
        ch.in_cons = &s_cons[cbase + j - 1];
        ch.in_base = r * T;
      } else {
        ch.in_prog = &s_prog[cbase + GS - 1];
        ch.grow_in = wrap;
        ch.in_base = (r - 1) * T;   // the wrap row was written in the previous round
      }
      ch.out_ring = j < GS - 1;
      if (j < GS - 1) {
        ch.out_sring = static_cast<uint32_t>(__cvta_generic_to_shared(rings + (size_t)(lbase + j) * LONG_RING));
        ch.out_cons = &s_cons[cbase + j];
      } else {
        ch.grow_out = wrap;         // only reached when ns > GS: the round wrap
      }
      ch.out_prog = &s_prog[cbase + j];
      const void* pstream = NIB ? static_cast<const void*>(reinterpret_cast<const uint8_t*>(a.stream) + pr.off)
                                : static_cast<const void*>(a.stream + pr.off);
      strip_pass<32, LR, true, false, LONG_US, NIB>(myprof, a.LSL, a.LBL, pstream, pr.len, T, lane, rd, wr,
                                                   nullptr, nullptr, ch, a.code_pad2, a.nGe, a.nGsGe, best);
    }
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) best = __vmaxs2(best, __shfl_xor_sync(FULL, best, o));
    if (lane == 0) s_best[warp] = best;
    __syncthreads();
    if (tid < P) {
      const int pj = li.y * P + tid;
      if (pj < d.n_long) {
        const PairRec pq = a.pairs[pj];
        uint32_t b = 0;
        for (int w = tid * GS; w < tid * GS + GS; ++w) b = __vmaxs2(b, s_best[w]);
        const int v0 = int(int16_t(b & 0xffffu)), v1 = int(int16_t(b >> 16));
        d.scores[pq.id0] = v0;
        if (v0 >= a.thr) flag_overflow(a.ovf_count, a.ovf, a.ovf_cap, d.qidx, pj, 0);
        if (pq.id1 >= 0) {
          d.scores[pq.id1] = v1;
          if (v1 >= a.thr) flag_overflow(a.ovf_count, a.ovf, a.ovf_cap, d.qidx, pj, 1);
        }
      }
    }
    __syncthreads();
  }
}
// The short-pair kernel: one persistent launch per short-pair mode (query pairs,
// single query), one (G, R) per launch, its own register budget (the query-pair
// form keeps R = 32 rows per lane at 128 registers, 2 CTAs per SM).
template <int G, int R, int NT, bool Q2, bool CG = false, bool NIB = false>
__global__ void __launch_bounds__(NT, 2) short_kernel(ShortArgs as) {
  extern __shared__ __align__(128) uint8_t smem[];
  __shared__ int s_item;
  __shared__ __align__(8) uint64_t s_mbar[2];
  int loaded = -1;  // (slot << 16 | strip) of the strip profile in shared memory (CTA-uniform)
  ProfStage ps{{-1, -1}, 0u, 0u, s_mbar};
  if (Q2 && threadIdx.x == 0) {
    mbar_init(s_mbar, 1);
    mbar_init(s_mbar + 1, 1);
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
  }
  for (;;) {
    if (threadIdx.x == 0) s_item = atomicAdd(as.work_counter, 1);
    __syncthreads();
    const int item = s_item;
    __syncthreads();
    if (item >= as.n_items) break;
    short_item<G, R, NT, Q2, CG, NIB>(as, item, smem, loaded, ps);
  }
}

// A long item as an out-of-line call: the combined single-query kernel below keeps
// the short path's register allocation apart from it (inlined: C2 -4 to -8 %,
// profiles/r02_ab_combined_forms.txt).
template <bool NIB>
__device__ __noinline__ void long_item_call(const LongArgs& a, int item, uint8_t* smem, LongShared& sh) {
  long_item<NIB, LONG_R_COMBINED>(a, item, smem, sh);
}

// Single-query searches with long pairs (C1/C2): ONE persistent launch, the long
// items first (costliest), then the short items, so the longest pairs start at
// once and the SMs that finish them move on to short items.
template <int G, int R, int NT, bool NIB = false, bool CG = false>
__global__ void __launch_bounds__(NT, 2) combined_m0_kernel(ShortArgs as, LongArgs al) {
  extern __shared__ __align__(128) uint8_t smem[];
  __shared__ int s_item;
  __shared__ LongShared sh;
  int loaded = -1;
  ProfStage ps{{-1, -1}, 0u, 0u, nullptr};  // (single-query items copy their profile by hand)
  const int n_items = al.n_items + as.n_items;
  for (;;) {
    if (threadIdx.x == 0) s_item = atomicAdd(as.work_counter, 1);
    __syncthreads();
    const int item = s_item;
    __syncthreads();
    if (item >= n_items) break;
    if (item < al.n_items) {
      long_item_call<NIB>(al, item, smem, sh);
      loaded = -1;  // the long item overwrote the strip profile
    } else {
      short_item<G, R, NT, false, CG, NIB>(as, item - al.n_items, smem, loaded, ps);
    }
  }
}

// The long-pair (intra-task) kernel: one persistent launch, costliest items first.
// When short pairs are scored too it runs concurrently with the short-pair kernel
// on a side stream, one CTA per SM (a shared-memory request that leaves no room
// for a short-pair CTA), so the co-resident short warps do not stretch the
// critical path of the longest pairs.
template <bool NIB>
__global__ void __launch_bounds__(LONG_W * 32, 1) long_kernel(LongArgs al) {
  extern __shared__ __align__(128) uint8_t smem[];
  __shared__ int s_item;
  __shared__ LongShared sh;
  for (;;) {
    if (threadIdx.x == 0) s_item = atomicAdd(al.work_counter, 1);
    __syncthreads();
    const int item = s_item;
    __syncthreads();
    if (item >= al.n_items) break;
    long_item<NIB, LONG_R>(al, item, smem, sh);
  }
}

// ---------------------------------------------------------------------------
// Instantiation tables.
typedef void (*short_fn)(ShortArgs);
#define SW_GEOM_CASES(X)                                                           \
  X(4, 8) X(4, 12) X(4, 16) X(4, 20) X(4, 24) X(4, 28) X(4, 32)                    \
  X(8, 8) X(8, 12) X(8, 16) X(8, 20) X(8, 24) X(8, 28) X(8, 32)                    \
  X(16, 8) X(16, 12) X(16, 16) X(16, 20) X(16, 24) X(16, 28) X(16, 32)             \
  X(32, 8) X(32, 12) X(32, 16) X(32, 20) X(32, 24) X(32, 28) X(32, 32)

// constant-gap (Gs 10, Ge 2) instantiations of the geometries the cost model picks
// for Swiss-Prot-like databases
#define SW_CG_CASES(X) X(4, 32) X(4, 24) X(8, 32) X(8, 24) X(4, 16) X(8, 16)
// 4-bit (nucleotide) database streams: a geometry subset (the cost model picks among them)
#define SW_NIB_CASES(X) X(4, 16) X(4, 24) X(4, 32) X(8, 16) X(8, 24) X(16, 12) X(16, 24) X(32, 8) X(32, 16)

// one-group CTAs for latency-bound single-query searches
#define SW_SMALL_CASES(X) X(32, 8) X(32, 12) X(32, 16)

static short_fn pick_short(int mode, int G, int R, bool cg = false, bool nib = false, int nt = SCORE_NT) {
  if (nt == 32) {
    if (mode != 0 || nib) return nullptr;
#define X(g, r) if (G == g && R == r) return short_kernel<g, r, 32, false>;
    SW_SMALL_CASES(X)
#undef X
    return nullptr;
  }
  if (nib) {
    if (mode == 1) {
#define X(g, r) if (G == g && R == r) return short_kernel<g, r, SCORE_NT, true, false, true>;
      SW_NIB_CASES(X)
#undef X
    } else {
#define X(g, r) if (G == g && R == r) return short_kernel<g, r, SCORE_NT, false, false, true>;
      SW_NIB_CASES(X)
#undef X
    }
    return nullptr;
  }
  if (cg && mode == 1) {
#define X(g, r) if (G == g && R == r) return short_kernel<g, r, SCORE_NT, true, true>;
    SW_CG_CASES(X)
#undef X
  }
  if (cg && mode == 0) {
#define X(g, r) if (G == g && R == r) return short_kernel<g, r, SCORE_NT, false, true>;
    SW_CG_CASES(X)
#undef X
  }
  if (mode == 1) {
#define X(g, r) if (G == g && R == r) return short_kernel<g, r, SCORE_NT, true>;
    SW_GEOM_CASES(X)
#undef X
  } else {
#define X(g, r) if (G == g && R == r) return short_kernel<g, r, SCORE_NT, false>;
    SW_GEOM_CASES(X)
#undef X
  }
  return nullptr;
}

bool short_config_supported(int mode, int G, int R, bool nib, int nt) {
  return pick_short(mode, G, R, false, nib, nt) != nullptr;
}

static int occupancy(const void* f, int threads, int smem_bytes) {
  if (smem_bytes > 48 * 1024) cudaFuncSetAttribute(f, cudaFuncAttributeMaxDynamicSharedMemorySize, smem_bytes);
  int n = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&n, f, threads, smem_bytes) != cudaSuccess) return 0;
  return n;
}

static short_fn pick_short_or_plain(int mode, int G, int R, bool cg, bool nib, int nt) {
  if (nt != SCORE_NT) return pick_short(mode, G, R, false, nib, nt);
  short_fn f = pick_short(mode, G, R, cg && !nib, nib);
  return (f || nib) ? f : pick_short(mode, G, R);
}

int short_max_ctas_per_sm(int mode, int G, int R, int smem_bytes, bool cg, bool nib, int nt) {
  short_fn f = pick_short_or_plain(mode, G, R, cg, nib, nt);
  return f ? occupancy(reinterpret_cast<const void*>(f), nt, smem_bytes) : 0;
}

cudaError_t launch_short(int mode, int G, int R, int grid, int smem_bytes, const ShortArgs& a, cudaStream_t st,
                         bool cg, bool nib, int nt) {
  short_fn f = pick_short_or_plain(mode, G, R, cg, nib, nt);
  if (!f) return cudaErrorInvalidValue;
  if (smem_bytes > 48 * 1024) {
    cudaError_t e = cudaFuncSetAttribute(f, cudaFuncAttributeMaxDynamicSharedMemorySize, smem_bytes);
    if (e != cudaSuccess) return e;
  }
  f<<<grid, nt, smem_bytes, st>>>(a);
  return cudaGetLastError();
}

typedef void (*combined_fn)(ShortArgs, LongArgs);
static combined_fn pick_combined(int G, int R, bool nib, bool cg) {
  if (cg && !nib) {
#define X(g, r) if (G == g && R == r) return combined_m0_kernel<g, r, SCORE_NT, false, true>;
    SW_CG_CASES(X)
#undef X
  }
  if (nib) {
#define X(g, r) if (G == g && R == r) return combined_m0_kernel<g, r, SCORE_NT, true>;
    SW_NIB_CASES(X)
#undef X
    return nullptr;
  }
#define X(g, r) if (G == g && R == r) return combined_m0_kernel<g, r, SCORE_NT>;
  SW_GEOM_CASES(X)
#undef X
  return nullptr;
}

int combined_max_ctas_per_sm(int G, int R, int smem_bytes, bool nib, bool cg) {
  combined_fn f = pick_combined(G, R, nib, cg);
  return f ? occupancy(reinterpret_cast<const void*>(f), SCORE_NT, smem_bytes) : 0;
}

cudaError_t launch_combined(int G, int R, int grid, int smem_bytes, const ShortArgs& as, const LongArgs& al,
                            cudaStream_t st, bool nib, bool cg) {
  combined_fn f = pick_combined(G, R, nib, cg);
  if (!f) return cudaErrorInvalidValue;
  if (smem_bytes > 48 * 1024) {
    cudaError_t e = cudaFuncSetAttribute(f, cudaFuncAttributeMaxDynamicSharedMemorySize, smem_bytes);
    if (e != cudaSuccess) return e;
  }
  f<<<grid, SCORE_NT, smem_bytes, st>>>(as, al);
  return cudaGetLastError();
}

int long_max_ctas_per_sm(int smem_bytes, bool nib) {
  return occupancy(nib ? reinterpret_cast<const void*>(long_kernel<true>) : reinterpret_cast<const void*>(long_kernel<false>),
                   LONG_W * 32, smem_bytes);
}

cudaError_t launch_long(int grid, int smem_bytes, const LongArgs& a, cudaStream_t st, bool nib) {
  auto f = nib ? long_kernel<true> : long_kernel<false>;
  if (smem_bytes > 48 * 1024) {
    cudaError_t e = cudaFuncSetAttribute(f, cudaFuncAttributeMaxDynamicSharedMemorySize, smem_bytes);
    if (e != cudaSuccess) return e;
  }
  f<<<grid, LONG_W * 32, smem_bytes, st>>>(a);
  return cudaGetLastError();
}

// ---------------------------------------------------------------------------
// Exact int32 re-score of flagged pairs.  The same chained
// wavefront as the long-pair mode, one problem per lane in int32 (s32 DPX),
// S read from a shared 33x33 matrix.  A flagged pair (entry) is split over K
// CTAs, one round each: CTA c of entry e holds strips W*c .. W*c + W-1 (32
// lanes x RESCORE_R rows each), chained warp to warp through per-CTA link rows
// + shared counters and CTA c-1 -> c through a global row + GPU-scope counter.
// Every wait targets an item taken earlier (CTA c-1 of the same entry, or the
// last users of a reused row block), so any grid size and any co-residency is
// deadlock-free.  The number of entries is read here, on the device: the host
// enqueues this kernel unconditionally and never waits for the scoring kernel.
// Row blocks are reused: entry e uses block e % ne_slots, after the ne_slots-
// earlier entry's K CTAs are done; counters carry (entry + 1) in their high
// word, so a stale value of the block's previous entry never satisfies a wait.
__device__ __forceinline__ unsigned long long ld_acquire_gpu_u64(const unsigned long long* p) {
  unsigned long long v;
  asm volatile("ld.acquire.gpu.global.b64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void st_release_gpu_u64(unsigned long long* p, unsigned long long v) {
  asm volatile("st.release.gpu.global.b64 [%0], %1;" :: "l"(p), "l"(v) : "memory");
}

// R rows per lane: 4 when every query has fewer than 2^11 strips of 128 rows (the
// (strip << 20) counters), else 8 -- the critical path is the pair's column count plus
// its strips x the per-strip lag, so shorter strips win (C4: 13.3 vs 14.9 ms).
template <int R>
__global__ void __launch_bounds__(RESCORE_WARPS * 32) rescore_kernel(RescoreArgs a) {
  constexpr int W = RESCORE_WARPS;
  constexpr int SW = 33;  // matrix row stride (PAD = alpha <= 32)
  __shared__ int32_t sm[SW * SW];
  __shared__ int s_prog[W];
  __shared__ int s_best[W];
  __shared__ int s_item;
  for (int i = threadIdx.x; i < SW * SW; i += blockDim.x) {
    const int x = i / SW, y = i % SW;
    sm[i] = (x < a.alpha && y < a.alpha) ? int(a.matrix[x * a.alpha + y]) : int(PAD_SCORE);
  }
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const bool lead = lane == 0, tail = lane == 31;
  int2* __restrict__ links = a.bbuf + (size_t)blockIdx.x * W * a.bcap;
  const int K = a.K;
  const int n_entries = min(*(volatile const int*)a.ovf_count, a.ovf_cap);
  const int n_items = n_entries * K;
  const int pad = a.alpha;
  const int nGe = -a.Ge, nGsGe = -(a.Gs + a.Ge);
  for (;;) {
    __syncthreads();
    if (threadIdx.x == 0) s_item = atomicAdd(a.work_counter, 1);
    if (threadIdx.x < W) { s_prog[threadIdx.x] = -1; s_best[threadIdx.x] = 0; }
    __syncthreads();
    const int item = s_item;
    if (item >= n_items) break;
    const int e = item / K, c = item - e * K;
    const OvfRec o = a.ovf[e];
    const PairRec pr = a.pairs[o.pair];
    const uint8_t* qc = a.qcodes + a.qoff[o.q];
    const int m = int(a.qoff[o.q + 1] - a.qoff[o.q]);
    const int L = pr.len;
    const int half = o.half;
    const int nstrips = (m + 32 * R - 1) / (32 * R);
    const int T = L + 32;
    const uint2 padw = pad_codes4(pad, a.nib);
    const int blk = e % a.ne_slots;
    int2* grow = a.grows + (int64_t)blk * K * a.bcap;
    unsigned long long* gflag = a.gflags + (int64_t)blk * K;
    const unsigned long long gen = (unsigned long long)(e + 1) << 32;
    const int j = W - 1 - warp;  // producers on higher warp ids (see long_kernel)
    const int s = W * c + j;
    // the block's previous entry must be finished before this CTA writes its row
    if (c + 1 < K && e >= a.ne_slots && warp == 0) {
      if (lane == 0)
        while (atomicAdd(a.done + (e - a.ne_slots), 0) < K) __nanosleep(256);
      __syncwarp();
    }
    __syncthreads();
    int best = 0;
    if (s < nstrips) {
      const bool rd = s > 0, wr = s + 1 < nstrips;
      const bool in_gpu = (j == 0 && c > 0), out_gpu = (j == W - 1 && c + 1 < K);
      const int2* rp = in_gpu ? grow + (int64_t)(c - 1) * a.bcap : links + (size_t)(j > 0 ? j - 1 : 0) * a.bcap;
      int2* wp = out_gpu ? grow + (int64_t)c * a.bcap : links + (size_t)j * a.bcap;
      const int in_base = (s - 1) << 20, out_base = s << 20;
      int seen = -1;
      auto wait_in = [&](int need) {
        if (seen >= need) return;
        for (;;) {
          int v = 0;
          if (lead) {
            if (in_gpu) {
              const unsigned long long x = ld_acquire_gpu_u64(gflag + (c - 1));
              v = (x >> 32) == (unsigned long long)(e + 1) ? int(x & 0xffffffffu) : -1;
            } else {
              v = ld_acquire_cta(&s_prog[j - 1]);
            }
          }
          v = __shfl_sync(FULL, v, 0);
          if (v >= need) { seen = v; break; }
          __nanosleep(in_gpu ? 256 : 64);  // (0 / 32 ns measured equal on C4, profiles/r02_ab_rescore_sleep.txt)
        }
        if (in_gpu) __threadfence();
      };
      rp += 31;
      int qr[R], Hl[R], E[R];
#pragma unroll
      for (int rr = 0; rr < R; ++rr) {
        const int row = s * 32 * R + lane * R + rr;
        qr[rr] = (row < m ? int(qc[row]) : pad) * SW;
        Hl[rr] = 0;
        E[rr] = 0;
      }
      int hdiag = 0, sH = 0, sF = 0, sC = pad;
      const int2 z2 = make_int2(0, 0);
      uint2 cw = padw;
      int2 tb0 = z2, tb1 = z2, tb2 = z2, tb3 = z2;
      if (rd && L > 0) wait_in(in_base + min(4 + 31 + RESCORE_LAG, L + 32));
      if (lead && L > 0) {
        cw = load_codes4(a.stream, pr.off, 0, a.nib);
        if (rd) { tb0 = __ldcg(rp + 0); tb1 = __ldcg(rp + 1); tb2 = __ldcg(rp + 2); tb3 = __ldcg(rp + 3); }
      }
      __syncwarp();
      for (int t0 = 0; t0 < T; t0 += 4) {
        const uint2 cwc = cw;
        const int2 c0 = tb0, c1 = tb1, c2 = tb2, c3 = tb3;
        if (rd && t0 + 4 < L) wait_in(in_base + min(t0 + 8 + 31 + RESCORE_LAG, L + 32));
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
          int hd = hdiag;
          hdiag = rH;
          int F = rF;
          int dprev = 0;
#pragma unroll
          for (int rr = 0; rr < R; ++rr) {
            const int dg = hd + sm[qr[rr] + rC];                        // FMA pipe
            const int h = __vimax3_s32(dg, E[rr], F);                    // Eq. (2) (E, F >= 0)
            hd = Hl[rr];
            Hl[rr] = h;
            const int tt = h + nGsGe;
            E[rr] = __viaddmax_s32_relu(E[rr], nGe, tt);                 // Eq. (3)
            F = __viaddmax_s32_relu(F, nGe, tt);                         // Eq. (4)
            if (rr & 1) best = __vimax3_s32(best, dprev, dg);            // max D = max H
            else dprev = dg;
          }
          sH = Hl[R - 1];
          sF = F;
          sC = rC;
          if (wr && tail) __stcg(wp + t0 + jj, make_int2(sH, sF));
        }
        if (wr && tail) {
          if (!out_gpu) st_release_cta(&s_prog[j], out_base + t0 + 4);
          else if (((t0 >> 2) & 3) == 3 || t0 + 4 >= T)
            st_release_gpu_u64(gflag + c, gen | (unsigned long long)(unsigned)(out_base + t0 + 4));
        }
      }
    }
#pragma unroll
    for (int off = 16; off > 0; off >>= 1) best = max(best, __shfl_xor_sync(FULL, best, off));
    if (lane == 0) s_best[warp] = best;
    __syncthreads();
    if (threadIdx.x == 0) {
      int b = 0;
      for (int w = 0; w < W; ++w) b = max(b, s_best[w]);
      const int id = o.half ? pr.id1 : pr.id0;
      if (K == 1) {
        a.scores[(int64_t)o.q * a.n_seqs + id] = b;
        atomicAdd(a.done + e, 1);
      } else {
        atomicMax(a.acc + e, b);
        __threadfence();
        if (atomicAdd(a.done + e, 1) == K - 1) {
          __threadfence();
          a.scores[(int64_t)o.q * a.n_seqs + id] = atomicAdd(a.acc + e, 0);
        }
      }
    }
  }
}

cudaError_t launch_rescore(int grid, const RescoreArgs& a, cudaStream_t st, int rows) {
  if (rows == 4) rescore_kernel<4><<<grid, RESCORE_WARPS * 32, 0, st>>>(a);  // persistent; K CTAs per flagged pair
  else rescore_kernel<RESCORE_R><<<grid, RESCORE_WARPS * 32, 0, st>>>(a);
  return cudaGetLastError();
}

// Mapped DBs (sw_load_db_mapped): the empty sequences' output columns are zeroed
// individually, because the rest of each row belongs to other shards.
__global__ void zero_columns_kernel(int32_t* scores, int64_t stride, int nq, const int64_t* cols, int64_t ncols) {
  const int64_t n = int64_t(nq) * ncols;
  for (int64_t x = blockIdx.x * int64_t(blockDim.x) + threadIdx.x; x < n; x += int64_t(gridDim.x) * blockDim.x)
    scores[(x / ncols) * stride + cols[x % ncols]] = 0;
}

cudaError_t launch_zero_columns(int32_t* scores, int64_t stride, int nq, const int64_t* cols, int64_t ncols,
                                cudaStream_t st) {
  const int64_t n = int64_t(nq) * ncols;
  if (n <= 0) return cudaSuccess;
  zero_columns_kernel<<<int(std::min<int64_t>((n + 255) / 256, 1024)), 256, 0, st>>>(scores, stride, nq, cols, ncols);
  return cudaGetLastError();
}

// Merge of gathered score blocks into scores[Q][N] in the caller's order (SURVEY
// 8(a) a8; the master's "merge").  Block b holds rows x cols
// int32 values at src + src_off (row-major), row i -> query rows[row_off + i],
// column k -> DB column cols[col_off + k].  One thread per element, grid-stride
// over a flat index; a small per-block prefix table locates the block.
__global__ void assemble_kernel(const int32_t* __restrict__ src, const AsmBlock* __restrict__ blocks, int n_blocks,
                                const int64_t* __restrict__ prefix, const int32_t* __restrict__ rows,
                                const int64_t* __restrict__ cols, int32_t* __restrict__ out, int64_t N) {
  const int64_t total = prefix[n_blocks];
  for (int64_t x = blockIdx.x * int64_t(blockDim.x) + threadIdx.x; x < total; x += int64_t(gridDim.x) * blockDim.x) {
    int lo = 0, hi = n_blocks - 1;  // the block holding element x: prefix[b] <= x < prefix[b+1]
    while (lo < hi) {
      const int mid = (lo + hi + 1) >> 1;
      if (prefix[mid] <= x) lo = mid; else hi = mid - 1;
    }
    const AsmBlock bk = blocks[lo];
    const int64_t e = x - prefix[lo];
    const int64_t i = e / bk.n_cols, k = e - i * bk.n_cols;
    out[int64_t(rows[bk.row_off + i]) * N + cols[bk.col_off + k]] = src[bk.src_off + e];
  }
}

cudaError_t launch_assemble(const int32_t* src, const AsmBlock* blocks, int n_blocks, const int64_t* prefix,
                            int64_t total, const int32_t* rows, const int64_t* cols, int32_t* out, int64_t N,
                            int sms, cudaStream_t st) {
  if (total <= 0) return cudaSuccess;
  const int grid = int(std::min<int64_t>((total + 255) / 256, int64_t(sms) * 8));
  assemble_kernel<<<grid, 256, 0, st>>>(src, blocks, n_blocks, prefix, rows, cols, out, N);
  return cudaGetLastError();
}

}  // namespace swdual
