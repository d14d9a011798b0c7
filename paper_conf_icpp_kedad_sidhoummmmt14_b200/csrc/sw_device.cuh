// Device-side building blocks of the Gotoh cell update on sm_100a DPX.
//
// Recurrences (sec. II.B, Eqs. (2)-(4), L178-194), s = query (rows i),
// t = database sequence (columns j):
//   H_ij = max(H_{i-1,j-1} + S_ij, E_ij, F_ij, 0)
//   E_ij = -Ge + max(E_{i,j-1}, H_{i,j-1} - Gs)
//   F_ij = -Ge + max(F_{i-1,j}, H_{i-1,j} - Gs)
// E and F are clamped at 0 (exact: H >= 0 absorbs any negative E/F, DESIGN.md
// reading R-9), so every stored value lies in [0, 32767] and the H maximum
// detects the only possible (upward) int16 wrap.
//
// Two independent problems share every 32-bit register (s16x2): the low half
// scores the query against DB sequence id0 of a pair, the high half against id1.
// Per cell pair: VIADDMNMX (Hdiag+S vs E) + VIMNMX (vs F) + VIADD.16x2 (H-Gs-Ge) +
// 2x VIADDMNMX.RELU (E', F') + 1/2 VIMNMX3 (running max) = 5.5 DPX lane-ops,
// plus one sign-extending PRMT that builds the (S[q_i][a], S[q_i][b]) word from
// the int8 query profile rows of the two DB letters a, b.
#pragma once
#include <cstdint>

namespace swdual {

__device__ __forceinline__ uint32_t prmt(uint32_t a, uint32_t b, uint32_t sel) {
  uint32_t d;
  asm("prmt.b32 %0, %1, %2, %3;" : "=r"(d) : "r"(a), "r"(b), "r"(sel));
  return d;
}

// Selector that turns int8 row j (0..3) of word a (letter of id0) and word b
// (letter of id1) into the s16x2 word (sext a_j, sext b_j): the msb of a PRMT
// selector nibble replicates the sign of the selected byte.
__host__ __device__ constexpr uint32_t pair_sel(int j) {
  return uint32_t(j) | (uint32_t(j | 8) << 4) | (uint32_t(4 + j) << 8) | (uint32_t((4 + j) | 8) << 12);
}

template <int R>
struct ProfUnit {
  static constexpr int BYTES = (R % 8 == 0) ? 8 : 4;  // LDS.64 or LDS.32 per letter
};

// Lane block size in bytes for R int8 rows: an odd number of load units so that
// consecutive lanes of a group hit distinct shared-memory banks.
__host__ __device__ constexpr int lane_block_bytes(int R) {
  return ((R % 8 == 0) ? (((R / 8) | 1) * 8) : (((R / 4) | 1) * 4));
}

// Shared-memory loads by 32-bit shared-window address (the profile pointers
// stay 32-bit: fewer registers than generic 64-bit pointers, no address
// rematerialisation in the hot loop).
__device__ __forceinline__ uint4 lds128(uint32_t a) {
  uint4 v;
  asm volatile("ld.shared.v4.u32 {%0, %1, %2, %3}, [%4];" : "=r"(v.x), "=r"(v.y), "=r"(v.z), "=r"(v.w) : "r"(a));
  return v;
}
__device__ __forceinline__ uint2 lds64(uint32_t a) {
  uint2 v;
  asm volatile("ld.shared.v2.u32 {%0, %1}, [%2];" : "=r"(v.x), "=r"(v.y) : "r"(a));
  return v;
}
__device__ __forceinline__ uint32_t lds32(uint32_t a) {
  uint32_t v;
  asm volatile("ld.shared.u32 %0, [%1];" : "=r"(v) : "r"(a));
  return v;
}

// Rows [R0, R1) of one column for one lane (a "sub-lane"; R0 = 0, R1 = R is
// the whole lane), ONE H buffer updated in place: the diagonal term of row r+1,
// D_{r+1} = H_{r,j-1} + S, is formed BEFORE H[r] is overwritten with H_{r,j},
// so the old value dies as the new one is born and H[r] keeps one register
// across columns (no second buffer, no moves).
//   H[r]   : in H_{r,j-1}, out H_{r,j}
//   E[r]   : in E_{r,j},   out E_{r,j+1}
//   hdiag  : in H_{R0-1, j-1}, out H_{R0-1, j}  (top boundary of the previous column)
//   Hio    : in H_{R0-1, j} (from above), out H_{R1-1, j}
//   Fio    : in F_{R0, j},                out F_{R1, j}
// Q2 = false: pa / pb are the shared addresses of the int8 profile rows of the
//   two DB letters of a pair (one per s16x2 half), combined per row by a
//   sign-extending PRMT.
// Q2 = true:  pa addresses s16x2 profile words (two queries, one DB letter).
// US: bytes between consecutive load units of one lane (= the unit size for the
// lane-blocked layout; G * unit for the unit-interleaved long-mode layout).
template <int R, int R0, int R1, bool Q2, int US = (Q2 ? 16 : ((R % 8 == 0) ? 8 : 4))>
__device__ __forceinline__ void gotoh_rows_inplace(uint32_t (&H)[R], uint32_t (&E)[R], uint32_t& best,
                                                   uint32_t& hdiag, uint32_t pa, uint32_t pb, uint32_t& Hio,
                                                   uint32_t& Fio,
                                                   uint32_t nGe, uint32_t nGsGe) {
  static_assert(R0 % 4 == 0 && (R1 - R0) % 4 == 0 && R1 <= R, "row range must be 4-aligned");
  constexpr int N = R1 - R0;
  uint32_t sv[N];  // S(q_r, letter) for the rows of this sub-lane
  constexpr int UB = Q2 ? 4 : ((R % 8 == 0 && R0 % 8 == 0 && N % 8 == 0) ? 8 : 4);
#pragma unroll
  for (int u = R0 / UB; u < R1 / UB; ++u) {
    const int b = u * UB - R0;
    if constexpr (Q2) {
      const uint4 w = lds128(pa + u * US);
      sv[b] = w.x; sv[b + 1] = w.y; sv[b + 2] = w.z; sv[b + 3] = w.w;
    } else if constexpr (UB == 8) {
      const uint2 x = lds64(pa + u * US);
      const uint2 y = lds64(pb + u * US);
#pragma unroll
      for (int j = 0; j < 8; ++j) sv[b + j] = prmt(j < 4 ? x.x : x.y, j < 4 ? y.x : y.y, pair_sel(j & 3));
    } else {
      constexpr bool IL = US > 8;
      const int off = IL ? (u >> 1) * US + (u & 1) * 4 : u * 4;
      const uint32_t x = lds32(pa + off);
      const uint32_t y = lds32(pb + off);
#pragma unroll
      for (int j = 0; j < 4; ++j) sv[b + j] = prmt(x, y, pair_sel(j));
    }
  }
  uint32_t F = Fio;
  uint32_t dcur = __vadd2(hdiag, sv[0]);  // D of row R0: H_{R0-1, j-1} + S
  hdiag = Hio;
  uint32_t dprev = 0;
#pragma unroll
  for (int i = 0; i < N; ++i) {
    const int r = R0 + i;
    uint32_t dnext = 0;
    if (i + 1 < N) dnext = __vadd2(H[r], sv[i + 1]);  // reads H_{r, j-1} before it is replaced
    const uint32_t h = __vimax3_s16x2(dcur, E[r], F);   // Eq. (2) (E, F >= 0)
    H[r] = h;
    const uint32_t t = __vadd2(h, nGsGe);               // H - Gs - Ge
    E[r] = __viaddmax_s16x2_relu(E[r], nGe, t);         // Eq. (3)
    F = __viaddmax_s16x2_relu(F, nGe, t);               // Eq. (4)
    if (r & 1) best = __vimax3_s16x2(best, dprev, dcur);  // max over D = max over H
    else dprev = dcur;
    dcur = dnext;
  }
  Hio = H[R1 - 1];
  Fio = F;
}

// Profile values S(q_r, letter) of rows [R0, R1) for one lane (see gotoh_rows_inplace).
template <int R, int R0, int R1, bool Q2, int US>
__device__ __forceinline__ void load_rows(uint32_t (&sv)[R1 - R0], uint32_t pa, uint32_t pb) {
  constexpr int N = R1 - R0;
  constexpr int UB = Q2 ? 4 : ((R % 8 == 0 && R0 % 8 == 0 && N % 8 == 0) ? 8 : 4);
#pragma unroll
  for (int u = R0 / UB; u < R1 / UB; ++u) {
    const int b = u * UB - R0;
    if constexpr (Q2) {
      const uint4 w = lds128(pa + u * US);
      sv[b] = w.x; sv[b + 1] = w.y; sv[b + 2] = w.z; sv[b + 3] = w.w;
    } else if constexpr (UB == 8) {
      const uint2 x = lds64(pa + u * US);
      const uint2 y = lds64(pb + u * US);
#pragma unroll
      for (int j = 0; j < 8; ++j) sv[b + j] = prmt(j < 4 ? x.x : x.y, j < 4 ? y.x : y.y, pair_sel(j & 3));
    } else {
      constexpr bool IL = US > 8;
      const int off = IL ? (u >> 1) * US + (u & 1) * 4 : u * 4;
      const uint32_t x = lds32(pa + off);
      const uint32_t y = lds32(pb + off);
#pragma unroll
      for (int j = 0; j < 4; ++j) sv[b + j] = prmt(x, y, pair_sel(j));
    }
  }
}

// Both sub-lanes of a lane in one interleaved sweep: sub-lane 0 = rows [0, RH)
// of column t, sub-lane 1 = rows [RH, R) of column t-1 (its inputs hdiag1 /
// Hio1 / Fio1 are sub-lane 0's outputs of the previous step).  The two F
// chains are independent, so emitting their rows alternately hands the
// scheduler two ready instructions per dependency step.
template <int R, bool Q2, int US>
__device__ __forceinline__ void gotoh_rows_dual(uint32_t (&H)[R], uint32_t (&E)[R], uint32_t& best,
                                                uint32_t& hdiag0, uint32_t pa0, uint32_t pb0, uint32_t& Hio0,
                                                uint32_t& Fio0, uint32_t& hdiag1, uint32_t pa1, uint32_t pb1,
                                                uint32_t& Hio1, uint32_t& Fio1, uint32_t nGe, uint32_t nGsGe) {
  constexpr int RH = R / 2;
  static_assert(R % 8 == 0, "two sub-lanes of whole 4-row units");
  uint32_t s0[RH], s1[RH];
  load_rows<R, 0, RH, Q2, US>(s0, pa0, pb0);
  load_rows<R, RH, R, Q2, US>(s1, pa1, pb1);
  uint32_t F0 = Fio0, F1 = Fio1;
  uint32_t d0 = __vadd2(hdiag0, s0[0]);
  uint32_t d1 = __vadd2(hdiag1, s1[0]);
  hdiag0 = Hio0;
  hdiag1 = Hio1;
#pragma unroll
  for (int i = 0; i < RH; ++i) {
    const int r0 = i, r1 = RH + i;
    uint32_t n0 = 0, n1 = 0;
    if (i + 1 < RH) {  // next rows' diagonals read H_{r, j-1} before it is replaced
      n0 = __vadd2(H[r0], s0[i + 1]);
      n1 = __vadd2(H[r1], s1[i + 1]);
    }
    const uint32_t h0 = __vimax3_s16x2(d0, E[r0], F0);  // Eq. (2)
    const uint32_t h1 = __vimax3_s16x2(d1, E[r1], F1);
    H[r0] = h0;
    H[r1] = h1;
    const uint32_t t0 = __vadd2(h0, nGsGe);
    const uint32_t t1 = __vadd2(h1, nGsGe);
    E[r0] = __viaddmax_s16x2_relu(E[r0], nGe, t0);    // Eq. (3)
    E[r1] = __viaddmax_s16x2_relu(E[r1], nGe, t1);
    F0 = __viaddmax_s16x2_relu(F0, nGe, t0);          // Eq. (4)
    F1 = __viaddmax_s16x2_relu(F1, nGe, t1);
    best = __vimax3_s16x2(best, d0, d1);              // max over D = max over H
    d0 = n0;
    d1 = n1;
  }
  Hio0 = H[RH - 1];
  Fio0 = F0;
  Hio1 = H[R - 1];
  Fio1 = F1;
}

// Lane block of the query-pair profile: R 4-byte rows, rounded to an odd number
// of 16-byte units (bank-conflict-free LDS.128 across the 8 lanes of a phase).
__host__ __device__ constexpr int lane_block_bytes_q2(int R) { return (((R / 4) | 1) * 16); }

constexpr uint32_t FULL = 0xffffffffu;

// Progress counters of chained strips (shared memory, CTA-scope release/acquire).
__device__ __forceinline__ int ld_acquire_cta(const int* p) {
  int v;
  asm volatile("ld.acquire.cta.shared.b32 %0, [%1];"
               : "=r"(v) : "r"(static_cast<uint32_t>(__cvta_generic_to_shared(const_cast<int*>(p)))) : "memory");
  return v;
}
__device__ __forceinline__ void st_relaxed_cta(int* p, int v) {
  asm volatile("st.relaxed.cta.shared.b32 [%0], %1;"
               :: "r"(static_cast<uint32_t>(__cvta_generic_to_shared(p))), "r"(v) : "memory");
}
__device__ __forceinline__ void st_release_cta(int* p, int v) {
  asm volatile("st.release.cta.shared.b32 [%0], %1;"
               :: "r"(static_cast<uint32_t>(__cvta_generic_to_shared(p))), "r"(v) : "memory");
}

// ---------------------------------------------------------------------------
// Bulk asynchronous copies (TMA engine, cp.async.bulk) global -> shared memory,
// completion counted in bytes on an mbarrier.
__device__ __forceinline__ uint32_t smem_u32(const void* p) {
  return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}
__device__ __forceinline__ void mbar_init(uint64_t* m, uint32_t count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" :: "r"(smem_u32(m)), "r"(count) : "memory");
}
__device__ __forceinline__ void mbar_arrive_expect_tx(uint64_t* m, uint32_t bytes) {
  asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" :: "r"(smem_u32(m)), "r"(bytes) : "memory");
}
__device__ __forceinline__ void bulk_g2s(void* dst, const void* src, uint32_t bytes, uint64_t* m) {
  asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];"
               :: "r"(smem_u32(dst)), "l"(src), "r"(bytes), "r"(smem_u32(m)) : "memory");
}
__device__ __forceinline__ void mbar_wait(uint64_t* m, uint32_t parity) {
  asm volatile("{\n .reg .pred p;\n"
               "WAIT_%=:\n mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n"
               " @!p bra WAIT_%=;\n}" :: "r"(smem_u32(m)), "r"(parity) : "memory");
}
// generic-proxy accesses of shared memory before async-proxy (bulk copy) writes
__device__ __forceinline__ void fence_proxy_async_smem() {
  asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
}

// Pair-stream access of the int32 paths (re-score, sw_align): 4 columns per load,
// either 16-bit columns (uint2) or, for 4-bit nucleotide streams, bytes (uint32).
__device__ __forceinline__ uint2 load_codes4(const uint16_t* stream, int64_t off, int t0, int nib) {
  if (nib) return make_uint2(reinterpret_cast<const uint32_t*>(reinterpret_cast<const uint8_t*>(stream) + off)[t0 >> 2], 0u);
  return reinterpret_cast<const uint2*>(stream + off)[t0 >> 2];
}
// the letter of column jj (0..3) of a 4-column block, half 0 (id0) or 1 (id1)
__device__ __forceinline__ int code_of(uint2 cw, int jj, int half, int nib) {
  if (nib) return int((cw.x >> (8 * jj + 4 * half)) & 0xfu);
  const uint32_t w = (jj < 2) ? cw.x : cw.y;
  return int((((jj & 1) ? (w >> 16) : w) >> (8 * half)) & 0xffu);
}
__device__ __forceinline__ uint2 pad_codes4(int pad, int nib) {
  const uint32_t b = nib ? uint32_t(pad | (pad << 4)) : uint32_t(pad);
  const uint32_t w = b * 0x01010101u;
  return make_uint2(w, nib ? 0u : w);
}

// GPU-scope counters (sw_align's CTA-to-CTA chains of very tall pairs).
__device__ __forceinline__ int ld_acquire_gpu(const int* p) {
  int v;
  asm volatile("ld.acquire.gpu.global.b32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void st_release_gpu(int* p, int v) {
  asm volatile("st.release.gpu.global.b32 [%0], %1;" :: "l"(p), "r"(v) : "memory");
}

// Link of a chained strip (sw_align): the row above (read by lane 0) and this
// strip's bottom row (written by the last lane), each with a progress counter.
struct Link {
  int* in;        // counter of the producer of the row above (nullptr: none)
  int in_base;    // value the producer publishes before its first cell
  bool in_gpu;    // counter in global memory (other CTA)
  int* out;       // this strip's counter (nullptr: nobody consumes it)
  int out_base;
  bool out_gpu;
};

// Warp-uniform wait until a progress counter reaches `need` (one lane polls,
// the result is broadcast, so the warp stays converged and the shuffles that
// follow stay on the fast path).  `seen` caches the last value observed.
__device__ __forceinline__ void wait_progress(const Link& lk, int need, int& seen) {
  if (seen >= need) return;
  for (;;) {
    int v = 0;
    if ((threadIdx.x & 31) == 0) v = lk.in_gpu ? ld_acquire_gpu(lk.in) : ld_acquire_cta(lk.in);
    v = __shfl_sync(FULL, v, 0);
    if (v >= need) { seen = v; break; }
    __nanosleep(lk.in_gpu ? 256 : 64);
  }
  if (lk.in_gpu) __threadfence();  // lane 0 acquired; make the row visible to its later loads
}

}  // namespace swdual
