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

// Rows [R0, R1) of one column for one lane (a "sub-lane"; R0 = 0, R1 = R is
// the whole lane).
//   Hin[r] : H_{r,j-1} (previous column);  Hout[r] : out H_{r,j}  (the caller
//            alternates two buffers, so the diagonal needs no register moves)
//   E[r]   : in E_{r,j},   out E_{r,j+1}
//   hdiag  : in H_{R0-1, j-1}, out H_{R0-1, j}  (top boundary of the previous column)
//   Hio    : in H_{R0-1, j} (from above), out H_{R1-1, j}
//   Fio    : in F_{R0, j},                out F_{R1, j}
// Q2 = false: pa / pb point at the int8 profile rows of the two DB letters of a
//   pair (one per s16x2 half), combined per row by a sign-extending PRMT.
// Q2 = true:  pa points at s16x2 profile words (two queries, one DB letter).
template <int R, int R0, int R1, bool Q2>
__device__ __forceinline__ void gotoh_rows(const uint32_t (&Hin)[R], uint32_t (&Hout)[R], uint32_t (&E)[R],
                                           uint32_t& best, uint32_t& hdiag, const uint8_t* __restrict__ pa,
                                           const uint8_t* __restrict__ pb, uint32_t& Hio, uint32_t& Fio,
                                           uint32_t nGe, uint32_t nGsGe) {
  static_assert(R0 % 4 == 0 && (R1 - R0) % 4 == 0 && R1 <= R, "row range must be 4-aligned");
  uint32_t hd = hdiag;
  hdiag = Hio;
  uint32_t F = Fio;
  uint32_t dprev = 0;
  constexpr int UB = Q2 ? 4 : ((R % 8 == 0 && R0 % 8 == 0 && (R1 - R0) % 8 == 0) ? 8 : 4);  // rows per load
#pragma unroll
  for (int u = R0 / UB; u < R1 / UB; ++u) {
    uint32_t sv[UB];
    if constexpr (Q2) {
      const uint4 w = *reinterpret_cast<const uint4*>(pa + u * 16);
      sv[0] = w.x; sv[1] = w.y; sv[2] = w.z; sv[3] = w.w;
    } else if constexpr (UB == 8) {
      const uint2 x = *reinterpret_cast<const uint2*>(pa + u * 8);
      const uint2 y = *reinterpret_cast<const uint2*>(pb + u * 8);
#pragma unroll
      for (int j = 0; j < 8; ++j) sv[j] = prmt(j < 4 ? x.x : x.y, j < 4 ? y.x : y.y, pair_sel(j & 3));
    } else {
      const uint32_t x = *reinterpret_cast<const uint32_t*>(pa + u * 4);
      const uint32_t y = *reinterpret_cast<const uint32_t*>(pb + u * 4);
#pragma unroll
      for (int j = 0; j < 4; ++j) sv[j] = prmt(x, y, pair_sel(j));
    }
#pragma unroll
    for (int j = 0; j < UB; ++j) {
      const int r = u * UB + j;
      // Eq. (2): H = max(D, E, F) with D = Hdiag + S; E, F >= 0 so the 0 term is
      // implied.  D goes to the FMA pipe (VIADD.16x2) and feeds both the 3-input
      // max (VIMNMX3) and the running maximum: max over all D = max over all H
      // (E and F never exceed an earlier H), so the ALU pipe carries only
      // 1 + 1 + 1 + 1/2 = 3.5 ops per cell pair.
      const uint32_t dg = __vadd2(hd, sv[j]);
      const uint32_t h = __vimax3_s16x2(dg, E[r], F);
      hd = Hin[r];
      Hout[r] = h;
      const uint32_t t = __vadd2(h, nGsGe);                              // H - Gs - Ge
      E[r] = __viaddmax_s16x2_relu(E[r], nGe, t);                        // Eq. (3)
      F = __viaddmax_s16x2_relu(F, nGe, t);                              // Eq. (4)
      if (r & 1) best = __vimax3_s16x2(best, dprev, dg);
      else dprev = dg;
    }
  }
  Hio = Hout[R1 - 1];
  Fio = F;
}

// Lane block of the query-pair profile: R 4-byte rows, rounded to an odd number
// of 16-byte units (bank-conflict-free LDS.128 across the 8 lanes of a phase).
__host__ __device__ constexpr int lane_block_bytes_q2(int R) { return (((R / 4) | 1) * 16); }

}  // namespace swdual
