// SWDUAL hot-path kernels for sm_100a: query-profile build, the inter-task
// s16x2 DPX scoring kernel and the exact int32 re-score kernel.
//
// Inter-task kernel (the paper's "very coarse-grained" split
// across workers, with the "fine-grained" wavefront inside a
// worker, L202-216 / Fig. 2):
//   * a lane GROUP of G lanes scores one database pair (two length-neighbours,
//     one per s16x2 half) against one query;
//   * lane k of the group owns R consecutive query rows of the current strip
//     (strip height G*R rows); at step t it computes column t-k, so the group
//     sweeps the matrix as an anti-diagonal wave: the bottom row (H, F) and the
//     residue codes travel one lane down per step over warp shuffles;
//   * queries taller than one strip are done in passes; the last lane writes the
//     strip's bottom row to a per-group global boundary row that lane 0 reads
//     in the next pass;
//   * the int8 query profile of the current strip sits in shared memory;
//   * CTAs are persistent and take chunks of NT/G pairs from an atomic counter,
//     pairs sorted longest first.
#include <algorithm>
#include <cstdio>
#include "sw_internal.h"
#include "sw_device.cuh"

namespace swdual {

constexpr int8_t PAD_SCORE = -64;  // S[.][PAD] = S[PAD][.] <= 0 (reading R-12)
// Intra-task mode: a strip starts consuming the row above only once its
// producer is this many columns ahead, so producer and consumer warps of a
// chain run decoupled instead of in lock-step (the consumer then rarely waits).
constexpr int LINK_LAG = 64;
#ifndef SW_DUAL_LONG
#define SW_DUAL_LONG 0
#endif
#ifndef SW_DUAL
#define SW_DUAL 1  // both sub-lanes in one interleaved row sweep (gotoh_rows_dual)
#endif
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
        const int vb = mb < 0 ? 0 : (cb < alpha && a < alpha) ? M[cb * alpha + a] : PAD_SCORE;  // mb < 0: wide mode-0 profile
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

// DB codes of the current pair: every strip pass of an item re-reads them, so
// they could stay cached between strips (SW_CODES 0: streaming/evict-first,
// 1: default caching, 2: L2 evict_last).  Measured on config 3: 1 and 2 cut
// DRAM reads by 23% but run 1% slower (the kernel is ALU-bound); 0 is kept.
#ifndef SW_CODES
#define SW_CODES 0
#endif
// SW_Q2_ADDR 1: lane 0 turns the DB letter into its profile-row address once per
// column (PRMT + IMAD) and the lanes shuffle addresses instead of codes: 2 fewer
// ALU ops per column, but the extra live register doubles the spill at the
// 128-register cap -- measured -7.5% on config 3 (+0.4% on config 2); kept off.
// SW_SEL_IMAD 1: lane 0's three per-column selects (code, H, F of the row above)
// as integer multiply-adds (FMA pipe) instead of SEL (ALU pipe).  Measured -2% on
// config 3 (+0.8% on config 4): one ALU op traded for two issue slots; kept off.
// SW_T0_UNROLL: unroll factor of the 4-column block loop of a strip pass (2 measured
// -1.4% on config 3: more register moves and spill; kept at 1)
#ifndef SW_T0_UNROLL
#define SW_T0_UNROLL 1
#endif
#ifndef SW_SEL_IMAD
#define SW_SEL_IMAD 0
#endif
// a == 1 ? v : x, as x + a * (v - x) in two IMADs (a in {0, 1}; exact mod 2^32)
__device__ __forceinline__ uint32_t fma_sel(uint32_t a, uint32_t v, uint32_t x) {
  uint32_t d, r;
  asm("mad.lo.u32 %0, %1, 1, %2;" : "=r"(d) : "r"(v), "r"(0u - x));
  asm("mad.lo.u32 %0, %1, %2, %3;" : "=r"(r) : "r"(a), "r"(d), "r"(x));
  return r;
}
#ifndef SW_Q2_ADDR
#define SW_Q2_ADDR 0
#endif
#ifndef SW_BB_HINT
#define SW_BB_HINT 0
#endif
__device__ __forceinline__ uint4 ld_bb(const uint2* p, uint64_t pol) {
  if constexpr (SW_BB_HINT) return ld_l2_last(p, pol);
  else return *reinterpret_cast<const uint4*>(p);
}
__device__ __forceinline__ void st_bb(uint2* p, uint2 v, uint64_t pol) {
  if constexpr (SW_BB_HINT) st_l2_last(p, v, pol);
  else *p = v;
}
__device__ __forceinline__ uint2 ld_codes(const uint2* p, uint64_t pol) {
  if constexpr (SW_CODES == 0) return __ldcs(p);
  else if constexpr (SW_CODES == 1) return __ldg(p);
  else {
    uint2 v;
    asm volatile("ld.global.nc.L2::cache_hint.v2.u32 {%0, %1}, [%2], %3;" : "=r"(v.x), "=r"(v.y) : "l"(p), "l"(pol));
    return v;
  }
}

// One strip pass of a lane group over one pair: G lanes x R rows, columns
// streamed as an anti-diagonal wave.  Boundary rows: lane 0 reads the strip
// above at rp[c] (c = column, rp = row base + G - 1), lane G-1 writes this
// strip's bottom row at wp[t] (t = step).  LINKED: the row above is produced
// concurrently by another warp of the CTA (intra-task mode): lane 0 waits on
// its progress counter, lane G-1 publishes its own.
template <int R>
struct SubLanes {
  // Each lane runs V "sub-lanes" of R/V rows, the second one column behind the
  // first: two independent dependency chains per step (twice the ILP of the
  // row-to-row F chain), at the cost of a (V*G - 1)-column wave fill.
  static constexpr int V = (R % 8 == 0) ? 2 : 1;
};

template <int G, int R, bool LINKED, bool Q2 = false, int US = (Q2 ? 16 : ((R % 8 == 0) ? 8 : 4)), int PW = 0>
__device__ __forceinline__ void strip_pass(const uint8_t* sprof, int LS, int LB, const uint16_t* pstream, int L,
                                           int T, int k, bool rd, bool wr, const uint2* __restrict__ rp,
                                           uint2* __restrict__ wp, const Link& lk, uint32_t code_pad2,
                                           uint32_t nGe, uint32_t nGsGe, uint32_t& best, uint32_t shift = 0,
                                           uint32_t wmul = 0) {
  static_assert(!PW || (!Q2 && R % 8 == 0 && US == 16), "wide single-query profile: two sub-lanes, LDS.128 rows");
  constexpr int V = SubLanes<R>::V;
  constexpr int VG = V * G;   // width of the wave in sub-lanes
  constexpr int RH = R / V;   // rows per sub-lane
  uint32_t HA[R], E[R];
#pragma unroll
  for (int r = 0; r < R; ++r) { HA[r] = 0; E[r] = 0; }
  const uint32_t sbase = static_cast<uint32_t>(__cvta_generic_to_shared(sprof));
  // Q2 (SW_Q2_ADDR): the code that travels down the lanes is already the shared
  // address of the DB letter's profile row (lane-independent); lane 0 forms it
  // once per column with one PRMT (byte select) + IMAD, the others add laneoff.
  const uint32_t c0pad = (Q2 && SW_Q2_ADDR) ? sbase + (code_pad2 & 0xffu) * LS : code_pad2;
  uint32_t hdiag = 0, sH = 0, sF = 0, sC = c0pad;
  const uint2* __restrict__ codes = reinterpret_cast<const uint2*>(pstream);
  const uint32_t pad4 = code_pad2 | (code_pad2 << 16);
  const uint32_t laneoff = uint32_t(k) * LB;
  const bool lead = (k == 0), tail = (k == G - 1);
#if SW_SEL_IMAD
  const uint32_t lead01 = lead ? 1u : 0u;
#endif
  const uint2 z2 = make_uint2(0, 0);
  // second sub-lane: its inputs are the first sub-lane's outputs of the previous step
  uint32_t hdiag1 = 0, cH = 0, cF = 0, pC = c0pad;
  const uint32_t bsel = (shift >> 3) | 0x4440u;  // PRMT selector: byte `shift/8` of a column word, zero-extended
  const uint32_t pad_row = sbase + (code_pad2 & 0xffu) * LS + laneoff;
  uint32_t ppa = pad_row, ppb = pad_row;
  rp += VG - 1;  // sub-lane 0 of lane 0 reads column c at rp[c + VG - 1]
  // SW_BB_HINT 1: boundary rows with an L2 evict_last policy (DRAM writes -35%
  // on config 3, but 1% slower: the kernel is ALU-bound, DRAM is ~3% busy)
  const uint64_t pol = (SW_BB_HINT || SW_CODES == 2) ? l2_evict_last_policy() : 0;

  // lane 0 prefetch of block 0: 4 columns of codes and (if rd) 4 boundary cells.
  // L and t0 are multiples of 4, so one compare guards a whole block.
  uint2 cw = make_uint2(pad4, pad4);
  uint2 tb0 = z2, tb1 = z2, tb2 = z2, tb3 = z2;
  int seen = -1;
  if (LINKED && rd && L > 0) wait_progress(lk, lk.in_base + min(4 + VG - 1 + LINK_LAG, L + VG), seen);
  if (lead && L > 0) {
    cw = ld_codes(codes, pol);
    if (rd) {
      if (LINKED) { tb0 = __ldcg(rp + 0); tb1 = __ldcg(rp + 1); tb2 = __ldcg(rp + 2); tb3 = __ldcg(rp + 3); }
      else {  // rp is 32-byte aligned (see the bb base in inter_kernel)
        const uint4 x = ld_bb(rp, pol), y = ld_bb(rp + 2, pol);
        tb0 = make_uint2(x.x, x.y); tb1 = make_uint2(x.z, x.w); tb2 = make_uint2(y.x, y.y); tb3 = make_uint2(y.z, y.w);
      }
    }
  }
  __syncwarp();
#if SW_T0_UNROLL == 2
#pragma unroll 2
#endif
  for (int t0 = 0; t0 < T; t0 += 4) {
    const uint2 cwc = cw;
    const uint2 c0 = tb0, c1 = tb1, c2 = tb2, c3 = tb3;
    rp += 4;
    if (LINKED && rd && t0 + 4 < L) wait_progress(lk, lk.in_base + min(t0 + 8 + VG - 1 + LINK_LAG, L + VG), seen);
    if (lead) {
      if (t0 + 4 < L) {
        cw = ld_codes(codes + ((t0 + 4) >> 2), pol);
        if (rd) {
          if (LINKED) { tb0 = __ldcg(rp + 0); tb1 = __ldcg(rp + 1); tb2 = __ldcg(rp + 2); tb3 = __ldcg(rp + 3); }
          else {
            const uint4 x = ld_bb(rp, pol), y = ld_bb(rp + 2, pol);
            tb0 = make_uint2(x.x, x.y); tb1 = make_uint2(x.z, x.w); tb2 = make_uint2(y.x, y.y); tb3 = make_uint2(y.z, y.w);
          }
        }
      } else {
        cw = make_uint2(pad4, pad4);
        tb0 = z2; tb1 = z2; tb2 = z2; tb3 = z2;
      }
    }
    __syncwarp();
#pragma unroll
    for (int j = 0; j < 4; ++j) {
      uint32_t rH = __shfl_up_sync(FULL, sH, 1, G);
      uint32_t rF = __shfl_up_sync(FULL, sF, 1, G);
      uint32_t rC = __shfl_up_sync(FULL, sC, 1, G);
#if SW_SEL_IMAD
      {  // lane 0 takes the boundary row: x + lead01 * (v - x) on the FMA pipe instead of SEL (ALU)
        const uint32_t w = (j < 2) ? cwc.x : cwc.y;
        const uint32_t cl = (j & 1) ? (w >> 16) : (w & 0xffffu);
        const uint2 tv = (j == 0) ? c0 : (j == 1) ? c1 : (j == 2) ? c2 : c3;
        rC = fma_sel(lead01, cl, rC);
        rH = fma_sel(lead01, tv.x, rH);
        rF = fma_sel(lead01, tv.y, rF);
      }
#else
      if (lead) {
        const uint32_t w = (j < 2) ? cwc.x : cwc.y;
        if constexpr (Q2 && SW_Q2_ADDR) rC = sbase + prmt(w, 0u, bsel + ((j & 1) ? 2u : 0u)) * LS;
        else rC = (j & 1) ? (w >> 16) : (w & 0xffffu);
        const uint2 tv = (j == 0) ? c0 : (j == 1) ? c1 : (j == 2) ? c2 : c3;
        rH = tv.x;
        rF = tv.y;
      }
#endif
      uint32_t pa, pb;
      if constexpr (Q2 && SW_Q2_ADDR) {  // rC = profile-row address of the DB letter
        pa = rC + laneoff;
        pb = pa;
      } else if constexpr (Q2) {  // one DB sequence (byte `shift` of the pair word) against two queries
        pa = sbase + ((rC >> shift) & 0xffu) * LS + laneoff;
        pb = pa;
      } else {
        pa = sbase + (rC & 0xffu) * LS + laneoff;
        pb = sbase + (rC >> 8) * LS + laneoff;
      }
      if constexpr (V == 2) {
        uint32_t h1 = cH, f1 = cF;
        if constexpr (SW_DUAL && (Q2 || PW || (SW_DUAL_LONG && LINKED))) {  // measured: +3% for the query-pair mode, -2% with the PRMT (mode 0)
          gotoh_rows_dual<R, Q2, US, PW>(HA, E, best, hdiag, pa, pb, rH, rF, hdiag1, ppa, ppb, h1, f1, nGe, nGsGe,
                                         wmul);
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
        if (LINKED) __stcg(wp + j, make_uint2(sH, sF));
        else st_bb(wp + j, make_uint2(sH, sF), pol);
      }
    }
    wp += 4;
    if (LINKED && wr && tail) {  // release orders this lane's link writes before the counter
      if (!lk.out_gpu) st_release_cta(lk.out, lk.out_base + t0 + 4);
      else if (((t0 >> 2) & 3) == 3 || t0 + 4 >= T) st_release_gpu(lk.out, lk.out_base + t0 + 4);
    }
  }
}

__device__ __forceinline__ void emit_pair(const InterArgs& a, const QueryDesc& d, int p, const PairRec& pr,
                                          uint32_t best) {
  const int lo = int(int16_t(best & 0xffffu));
  const int hi = int(int16_t(best >> 16));
  d.scores[pr.id0] = lo;
  if (lo >= a.thr) {
    const int e = atomicAdd(a.ovf_count, 1);
    if (e < a.ovf_cap) a.ovf[e] = OvfRec{d.qidx, p, 0, 0};
  }
  if (pr.id1 >= 0) {
    d.scores[pr.id1] = hi;
    if (hi >= a.thr) {
      const int e = atomicAdd(a.ovf_count, 1);
      if (e < a.ovf_cap) a.ovf[e] = OvfRec{d.qidx, p, 1, 0};
    }
  }
}

// Persistent kernel over ALL queries of a search.  Work items, costliest first:
//   [0, Q*n_long): (query, LONG pair) -- scored by all W = NT/32 warps of the CTA
//     together (intra-task mode; the paper's fine-grained
//     wavefront across PEs, Fig. 2): warp w takes strips w, w+W, ...
//     of a 32-lane x LONG_R-row geometry, each strip consuming the bottom row of
//     the strip above through a global link row + shared progress counter;
//   then (query, CHUNK of NT/G short pairs) -- one pair per lane group
//     (inter-task mode).
// Queries are in descending length, pairs in descending length.
// PWK = 1: the variant whose single-query slots use the wide profile (a separate
// instantiation: its pair build needs more live registers, which must not raise
// the register allocation of the default kernel).
template <int G, int R, int NT, int PWK>
__device__ __forceinline__ void inter_body(InterArgs a) {
  extern __shared__ __align__(16) uint8_t smem[];
  // An item is either short or long, so the two uses share shared memory:
  uint8_t* sprof = smem;                         // short mode: the strip profile (bank-spread copies)
  uint8_t* lprof = smem + (SW_SMEM_UNION ? 0 : max(a.cstride[0] * (a.ncopy[0] - 1) + 128 + a.SB,
                                                    a.cstride[1] * (a.ncopy[1] - 1) + a.SB2));  // long mode: one a.SBL slot per warp
  __shared__ int s_item;
  __shared__ int s_prog[NT / 32];
  __shared__ uint32_t s_best[NT / 32];
  constexpr int NG = NT / G;
  constexpr int W = NT / 32;
  const int tid = threadIdx.x;
  const int k = tid & (G - 1);
  const int g = tid / G;
  const int lane = tid & 31, warp = tid >> 5;
  const int n_long_items = a.n_long_items;
  const int n_items = n_long_items + a.n_short_items;
  // per-group boundary row; offset so that &bb[V*G - 1] is 32-byte aligned (bcap % 4 == 0)
  constexpr int BB_PAD = (4 - (G * SubLanes<R>::V - 1) % 4) % 4;
  uint2* __restrict__ bb = a.bbuf + ((size_t)blockIdx.x * NG + g) * (size_t)a.bcap + BB_PAD;
  int loaded = -1;  // (query rank << 16 | strip) of the short profile in shared memory (CTA-uniform)

  for (;;) {
    if (tid == 0) s_item = atomicAdd(a.work_counter, 1);
    if (tid < W) { s_prog[tid] = -1; s_best[tid] = 0; }
    __syncthreads();
    const int item = s_item;
    if (item >= n_items) break;
    if (item < n_long_items) {
      loaded = -1;  // the long-mode slots overwrite the short strip profile
      // ---------------- long pair, superstrip k: W chained strips on this CTA's
      // warps; superstrips k-1 / k+1 of the same pair run on other CTAs
      int lo = 0, hi = a.n_queries - 1;
      while (lo < hi) {
        const int mid = (lo + hi + 1) >> 1;
        if (a.queries[mid].long_item_begin <= item) lo = mid; else hi = mid - 1;
      }
      const QueryDesc d = a.queries[lo];
      if (d.pairs_per_item > 1) {
        // ---- query shorter than W strips: P = W / S pairs per CTA, S warps per
        // pair (one strip each; upstream strips on higher warp ids)
        const int S = d.n_strips_long, P = d.pairs_per_item;
        const int grp = warp / S, jw = warp - grp * S;
        const int pidx = (item - d.long_item_begin) * P + grp;
        const bool active = grp < P && pidx < d.n_long;
        uint32_t best = 0;
        if (active) {
          const PairRec pr = a.pairs[pidx];
          const int s = S - 1 - jw;
          uint8_t* myprof = lprof + warp * a.SBL;
          {
            const uint4* src = reinterpret_cast<const uint4*>(d.prof_long + (size_t)s * a.SBL);
            uint4* dst = reinterpret_cast<uint4*>(myprof);
            for (int i = lane; i < a.SBL / 16; i += 32) dst[i] = __ldg(src + i);
          }
          __syncwarp();
          uint2* links = a.links + (size_t)blockIdx.x * W * a.lcap;
          Link lk{};
          const int wprod = warp + 1;  // the warp holding strip s-1 of this pair
          lk.in = &s_prog[s > 0 ? wprod : warp];
          lk.in_base = (s - 1) << 20;
          lk.out = &s_prog[warp];
          lk.out_base = s << 20;
          strip_pass<32, LONG_R, true, false, LONG_US>(myprof, a.LSL, a.LBL, a.stream + pr.off, pr.len,
                                       pr.len + 32 * SubLanes<LONG_R>::V, lane, s > 0, s + 1 < S,
                                       links + (size_t)(s > 0 ? wprod : warp) * a.lcap,
                                       links + (size_t)warp * a.lcap, lk, a.code_pad2, a.nGe, a.nGsGe, best);
        }
#pragma unroll
        for (int o = 16; o > 0; o >>= 1) best = __vmaxs2(best, __shfl_xor_sync(FULL, best, o));
        if (lane == 0) s_best[warp] = best;
        __syncthreads();
        if (tid < P) {
          const int pj = (item - d.long_item_begin) * P + tid;
          if (pj < d.n_long) {
            uint32_t b = 0;
            for (int w = tid * S; w < tid * S + S; ++w) b = __vmaxs2(b, s_best[w]);
            emit_pair(a, d, pj, a.pairs[pj], b);
          }
        }
        __syncthreads();
        continue;
      }
      const int K = d.n_super;               // CTAs sharing this pair
      const int64_t gstride = d.glink_stride;
      const int local = item - d.long_item_begin;
      const int pidx = local / K, c = local - pidx * K;
      const PairRec pr = a.pairs[pidx];
      const int T = pr.len + 32 * SubLanes<LONG_R>::V;
      uint32_t best = 0;
      uint8_t* myprof = lprof + warp * a.SBL;
      uint2* links = a.links + (size_t)blockIdx.x * W * a.lcap;
      uint2* grow = a.glinks + d.glink_base + a.lofs[pidx];
      int* gflag = a.gflags + d.flag_base + (int64_t)pidx * K;
      // Strips are dealt round-robin: round r of CTA c covers strips
      // W*(K*r + c) .. +W-1, one per warp.  Upstream strips run on the HIGHER
      // warp ids: the SMSP arbiter issues highest-warp-id first, so producers
      // keep their lead instead of being starved by consumers that caught up
      // and spin on the link counter.  The chain runs warp W-1 -> 0 inside a
      // CTA, then on to CTA c+1 (global boundary row + GPU-scope counter), and
      // from CTA K-1 back to CTA 0 for the next round.
      const int j = W - 1 - warp;
      const int ns = d.n_strips_long;
      for (int r = 0;; ++r) {
        const int s = W * (K * r + c) + j;   // strip index
        if (s >= ns) break;
        __syncwarp();
        {  // this warp's strip profile -> its own slot
          const uint4* src = reinterpret_cast<const uint4*>(d.prof_long + (size_t)s * a.SBL);
          uint4* dst = reinterpret_cast<uint4*>(myprof);
          for (int i = lane; i < a.SBL / 16; i += 32) dst[i] = __ldg(src + i);
        }
        __syncwarp();
        const bool rd = s > 0, wr = s + 1 < ns;
        Link lk{};
        const uint2* rp;
        uint2* wp;
        if (j > 0 || K == 1) {  // producer is a warp of this CTA (for K == 1: the last warp, previous round)
          const int jl = (j + W - 1) % W;
          rp = links + (size_t)jl * a.lcap;
          lk.in = &s_prog[jl];
        } else {                // producer is the last warp of CTA c-1 (or of CTA K-1, previous round)
          const int pc = (c + K - 1) % K;
          rp = grow + (int64_t)pc * gstride;
          lk.in = gflag + pc;
          lk.in_gpu = true;
        }
        lk.in_base = (s - 1) << 20;  // counters are monotone: (strip << 20) | cells written
        if (j < W - 1 || K == 1) {
          wp = links + (size_t)j * a.lcap;
          lk.out = &s_prog[j];
        } else {
          wp = grow + (int64_t)c * gstride;
          lk.out = gflag + c;
          lk.out_gpu = true;
        }
        lk.out_base = s << 20;
        strip_pass<32, LONG_R, true, false, LONG_US>(myprof, a.LSL, a.LBL, a.stream + pr.off, pr.len, T, lane, rd, wr, rp, wp, lk,
                                     a.code_pad2, a.nGe, a.nGsGe, best);
      }
#pragma unroll
      for (int o = 16; o > 0; o >>= 1) best = __vmaxs2(best, __shfl_xor_sync(FULL, best, o));
      if (lane == 0) s_best[warp] = best;
      __syncthreads();
      if (tid == 0) {
        uint32_t b = 0;
        for (int w = 0; w < W; ++w) b = __vmaxs2(b, s_best[w]);
        if (K == 1) {
          emit_pair(a, d, pidx, pr, b);
        } else {  // combine the superstrips' maxima; the last one to finish checks overflow
          atomicMax(d.scores + pr.id0, int(int16_t(b & 0xffffu)));
          if (pr.id1 >= 0) atomicMax(d.scores + pr.id1, int(int16_t(b >> 16)));
          __threadfence();
          if (atomicAdd(a.gdone + d.done_base + pidx, 1) == K - 1) {
            __threadfence();
            const int v0 = atomicAdd(d.scores + pr.id0, 0);
            const int v1 = pr.id1 >= 0 ? atomicAdd(d.scores + pr.id1, 0) : 0;
            if (v0 >= a.thr) {
              const int e = atomicAdd(a.ovf_count, 1);
              if (e < a.ovf_cap) a.ovf[e] = OvfRec{d.qidx, pidx, 0, 0};
            }
            if (pr.id1 >= 0 && v1 >= a.thr) {
              const int e = atomicAdd(a.ovf_count, 1);
              if (e < a.ovf_cap) a.ovf[e] = OvfRec{d.qidx, pidx, 1, 0};
            }
          }
        }
      }
    } else {
      // ---------------- short work: the host ordered all (slot, chunk) items of
      // the launch by critical path (strips x pair length), longest first
      const int2 sc = a.item_map[item - n_long_items];
      const int sl = sc.x;
      const SlotDesc d = a.slots[sl];
      const int chunk = sc.y;
      const bool q2 = d.mode == 1;
      constexpr bool wide = PWK != 0 && R % 8 == 0;  // mode 0 with the 32-bit (query-pair layout) profile
      int p, half = 0;
      if (q2) {  // chunk of NG half-pairs: DB sequence = one half of a pair
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
      if (q2 && half && pr.id1 < 0) valid = false;  // odd leftover pair has no high half
      int T = pr.len + G * SubLanes<R>::V;         // the last sub-lane finishes column len-1 at step T-2
      if (G < 32) T = __reduce_max_sync(FULL, T);  // warp-uniform trip count (shuffles)
      uint32_t best = 0;
      const bool l2 = q2 || wide;  // query-pair profile geometry
      const int SBx = l2 ? a.SB2 : a.SB;
      const int ncp = l2 ? a.ncopy[1] : a.ncopy[0], csx = l2 ? a.cstride[1] : a.cstride[0];
      const uint32_t skw = l2 ? 0u : a.cskew0;
      const int rs = d.res_stride;  // > 0: every strip of the slot resident (loaded once per slot)
      for (int s = 0; s < d.n_strips; ++s) {
        const int want = rs ? ((sl << 16) | 0xffff) : ((sl << 16) | s);
        if (want != loaded) {
          __syncthreads();
          if (rs) {
            for (int s2 = 0; s2 < d.n_strips; ++s2)
              for (int cp = 0; cp < ncp; ++cp)
                copy_strip(sprof + s2 * rs + copy_off(cp, csx, skw), d.prof + (size_t)s2 * SBx, SBx);
          } else {
            for (int cp = 0; cp < ncp; ++cp) copy_strip(sprof + copy_off(cp, csx, skw), d.prof + (size_t)s * SBx, SBx);
          }
          __syncthreads();
          loaded = want;
        }
        const uint8_t* gprof = sprof + (rs ? s * rs : 0) + copy_off(g & (ncp - 1), csx, skw);  // this group's bank-spread copy
        if (q2) {
          const StripInfo si = d.sinfo[s];
          const bool rd = s > 0 && si.keep != 0;
          if (rd && si.keep != FULL) {  // one half starts a new query: zero its half of the boundary row
            for (int c = k; c < T; c += G) {
              const uint2 v = bb[c];
              bb[c] = make_uint2(v.x & si.keep, v.y & si.keep);
            }
            __syncwarp();
          }
          strip_pass<G, R, false, true>(gprof, a.LS2, a.LB2, a.stream + pr.off, pr.len, T, k, rd,
                                        s + 1 < d.n_strips, bb, bb, Link{}, a.code_pad2,
                                        a.nGe, a.nGsGe, best, half ? 8u : 0u);
          if (si.emit0 >= 0 || si.emit1 >= 0) {  // a query of either half ends with this strip
            uint32_t bg = best;
#pragma unroll
            for (int o = G / 2; o > 0; o >>= 1) bg = __vmaxs2(bg, __shfl_xor_sync(FULL, bg, o, G));
            if (valid && k == 0) {
              const int id = half ? pr.id1 : pr.id0;
              if (si.emit0 >= 0) {
                const int v = int(int16_t(bg & 0xffffu));
                a.scores_all[(int64_t)si.emit0 * a.n_seqs + id] = v;
                if (v >= a.thr) {
                  const int e = atomicAdd(a.ovf_count, 1);
                  if (e < a.ovf_cap) a.ovf[e] = OvfRec{si.emit0, p, half, 0};
                }
              }
              if (si.emit1 >= 0) {
                const int v = int(int16_t(bg >> 16));
                a.scores_all[(int64_t)si.emit1 * a.n_seqs + id] = v;
                if (v >= a.thr) {
                  const int e = atomicAdd(a.ovf_count, 1);
                  if (e < a.ovf_cap) a.ovf[e] = OvfRec{si.emit1, p, half, 0};
                }
              }
            }
            best &= (si.emit0 >= 0 ? 0xffff0000u : 0xffffffffu) & (si.emit1 >= 0 ? 0x0000ffffu : 0xffffffffu);
          }
        } else {
          if constexpr (wide)
            strip_pass<G, R, false, false, 16, 1>(gprof, a.LS2, a.LB2, a.stream + pr.off, pr.len, T, k, s > 0,
                                                  s + 1 < d.n_strips, bb, bb, Link{}, a.code_pad2, a.nGe, a.nGsGe,
                                                  best, 0u, a.wmul);
          else
            strip_pass<G, R, false>(gprof, a.LS, a.LB, a.stream + pr.off, pr.len, T, k, s > 0, s + 1 < d.n_strips,
                                    bb, bb, Link{}, a.code_pad2, a.nGe, a.nGsGe, best);
        }
      }
      if (!q2) {  // mode 0: one query, both halves are DB sequences
#pragma unroll
        for (int o = G / 2; o > 0; o >>= 1) best = __vmaxs2(best, __shfl_xor_sync(FULL, best, o, G));
        if (valid && k == 0) {
          QueryDesc qd;
          qd.scores = d.scores0;
          qd.qidx = d.qidx0;
          emit_pair(a, qd, p, pr, best);
        }
      }
    }
    __syncthreads();
  }
}

template <int G, int R, int NT>
#ifdef SW_MINB  // experiments only: __launch_bounds__(NT, 1) lets ptxas take 225 registers (1 CTA/SM, -5% on config 3)
__global__ void __launch_bounds__(NT, SW_MINB) inter_kernel(InterArgs a) {
#else
__global__ void __launch_bounds__(NT) inter_kernel(InterArgs a) {
#endif
  inter_body<G, R, NT, 0>(a);
}
// the wide-profile variant, held to 2 CTAs/SM (128 registers) like the default
template <int G, int R, int NT>
__global__ void __launch_bounds__(NT, 2) inter_kernel_wide(InterArgs a) {
  inter_body<G, R, NT, 1>(a);
}

// ---------------------------------------------------------------------------
// Instantiation table.
#ifndef SW_INTER_NT
#define SW_INTER_NT 256
#endif
constexpr int INTER_NT = SW_INTER_NT;  // threads per CTA of the scoring kernel

#define SW_INTER_CASES(X)                                                          \
  X(4, 8) X(4, 12) X(4, 16) X(4, 20) X(4, 24) X(4, 28) X(4, 32)                    \
  X(8, 8) X(8, 12) X(8, 16) X(8, 20) X(8, 24) X(8, 28) X(8, 32)                    \
  X(16, 8) X(16, 12) X(16, 16) X(16, 20) X(16, 24) X(16, 28) X(16, 32)             \
  X(32, 8) X(32, 12) X(32, 16) X(32, 20) X(32, 24) X(32, 28) X(32, 32)

typedef void (*inter_fn)(InterArgs);

#define SW_WIDE_CASES(X) X(4, 24) X(8, 24) X(8, 16) X(16, 24) X(8, 32) X(4, 16)

static inter_fn pick_inter(int G, int R, int NT, int wide = 0) {
  if (NT != INTER_NT) return nullptr;
  if (wide) {
#define X(g, r) \
    if (G == g && R == r) return inter_kernel_wide<g, r, INTER_NT>;
    SW_WIDE_CASES(X)
#undef X
    return nullptr;
  }
#define X(g, r) \
  if (G == g && R == r) return inter_kernel<g, r, INTER_NT>;
  SW_INTER_CASES(X)
#undef X
  return nullptr;
}

bool inter_config_supported(int G, int R) { return pick_inter(G, R, INTER_NT) != nullptr; }
bool inter_wide_supported(int G, int R) { return pick_inter(G, R, INTER_NT, 1) != nullptr; }
int inter_block_threads() { return INTER_NT; }

int inter_max_ctas_per_sm(int G, int R, int NT, int smem_bytes, int wide) {
  inter_fn f = pick_inter(G, R, NT, wide);
  if (!f) return 0;
  if (smem_bytes > 48 * 1024)
    cudaFuncSetAttribute(f, cudaFuncAttributeMaxDynamicSharedMemorySize, smem_bytes);
  int n = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&n, f, NT, smem_bytes) != cudaSuccess) return 0;
  return n;
}

cudaError_t launch_inter(int G, int R, int NT, int grid, int smem_bytes, const InterArgs& a, cudaStream_t st,
                         int wide) {
  inter_fn f = pick_inter(G, R, NT, wide);
  if (!f) return cudaErrorInvalidValue;
  if (smem_bytes > 48 * 1024) {
    cudaError_t e = cudaFuncSetAttribute(f, cudaFuncAttributeMaxDynamicSharedMemorySize, smem_bytes);
    if (e != cudaSuccess) return e;
  }
  f<<<grid, NT, smem_bytes, st>>>(a);
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

__global__ void __launch_bounds__(RESCORE_WARPS * 32) rescore_kernel(RescoreArgs a) {
  constexpr int R = RESCORE_R;
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
    const uint32_t shift = o.half ? 8u : 0u;
    const int nstrips = (m + 32 * R - 1) / (32 * R);
    const int T = L + 32;
    const uint2* __restrict__ codes = reinterpret_cast<const uint2*>(a.stream + pr.off);
    const uint32_t padw = uint32_t(pad) * 0x01010101u;
    const int blk = e % a.ne_slots;
    int2* grow = a.grows + (int64_t)blk * K * a.bcap;
    unsigned long long* gflag = a.gflags + (int64_t)blk * K;
    const unsigned long long gen = (unsigned long long)(e + 1) << 32;
    const int j = W - 1 - warp;  // producers on higher warp ids (see inter_kernel)
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
          __nanosleep(in_gpu ? 256 : 64);
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
      uint2 cw = make_uint2(padw, padw);
      int2 tb0 = z2, tb1 = z2, tb2 = z2, tb3 = z2;
      if (rd && L > 0) wait_in(in_base + min(4 + 31 + RESCORE_LAG, L + 32));
      if (lead && L > 0) {
        cw = codes[0];
        if (rd) { tb0 = __ldcg(rp + 0); tb1 = __ldcg(rp + 1); tb2 = __ldcg(rp + 2); tb3 = __ldcg(rp + 3); }
      }
      __syncwarp();
      for (int t0 = 0; t0 < T; t0 += 4) {
        const uint2 cwc = cw;
        const int2 c0 = tb0, c1 = tb1, c2 = tb2, c3 = tb3;
        if (rd && t0 + 4 < L) wait_in(in_base + min(t0 + 8 + 31 + RESCORE_LAG, L + 32));
        if (lead) {
          if (t0 + 4 < L) {
            cw = codes[(t0 + 4) >> 2];
            if (rd) {
              tb0 = __ldcg(rp + t0 + 4); tb1 = __ldcg(rp + t0 + 5); tb2 = __ldcg(rp + t0 + 6); tb3 = __ldcg(rp + t0 + 7);
            }
          } else {
            cw = make_uint2(padw, padw);
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
            const uint32_t w = (jj < 2) ? cwc.x : cwc.y;
            rC = int(((jj & 1) ? (w >> 16) : w) >> shift) & 0xff;
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

cudaError_t launch_rescore(int grid, const RescoreArgs& a, cudaStream_t st) {
  rescore_kernel<<<grid, RESCORE_WARPS * 32, 0, st>>>(a);  // persistent; K CTAs per flagged pair
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
