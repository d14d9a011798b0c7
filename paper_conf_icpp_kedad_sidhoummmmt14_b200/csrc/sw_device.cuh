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

// One column of R rows for one lane.
//   Hin[r] : H_{r,j-1} (previous column);  Hl[r] : out H_{r,j}  (caller alternates
//            two buffers so the diagonal needs no register moves)
//   E[r]   : in E_{r,j},   out E_{r,j+1}
//   hdiag  : in H_{top-1, j-1}, out H_{top-1, j}  (top boundary of the previous column)
//   Hio    : in H_{top-1, j} (from the lane above), out H_{bottom, j}
//   Fio    : in F_{top, j},                        out F_{bottom+1, j}
template <int R>
__device__ __forceinline__ void gotoh_column(const uint32_t (&Hin)[R], uint32_t (&Hl)[R], uint32_t (&E)[R],
                                             uint32_t& best,
                                             uint32_t& hdiag, const uint8_t* __restrict__ pa,
                                             const uint8_t* __restrict__ pb, uint32_t& Hio, uint32_t& Fio,
                                             uint32_t nGe, uint32_t nGsGe) {
  uint32_t hd = hdiag;
  hdiag = Hio;
  uint32_t F = Fio;
  uint32_t hprev = 0;
  constexpr int UB = ProfUnit<R>::BYTES;
#pragma unroll
  for (int u = 0; u < R / UB; ++u) {
    uint32_t wa[UB / 4], wb[UB / 4];
    if constexpr (UB == 8) {
      const uint2 x = *reinterpret_cast<const uint2*>(pa + u * 8);
      const uint2 y = *reinterpret_cast<const uint2*>(pb + u * 8);
      wa[0] = x.x; wa[1] = x.y; wb[0] = y.x; wb[1] = y.y;
    } else {
      wa[0] = *reinterpret_cast<const uint32_t*>(pa + u * 4);
      wb[0] = *reinterpret_cast<const uint32_t*>(pb + u * 4);
    }
#pragma unroll
    for (int j = 0; j < UB; ++j) {
      const int r = u * UB + j;
      const uint32_t s = prmt(wa[j >> 2], wb[j >> 2], pair_sel(j & 3));
      // Eq. (2): H = max(D, E, F) with D = Hdiag + S; E, F >= 0 so the 0 term is
      // implied.  D goes to the FMA pipe (VIADD.16x2) and feeds both the 3-input
      // max (VIMNMX3) and the running maximum: max over all D = max over all H
      // (E and F never exceed an earlier H), so the ALU pipe carries only
      // 1 + 1 + 1 + 1/2 = 3.5 ops per cell pair.
      const uint32_t dg = __vadd2(hd, s);
      const uint32_t h = __vimax3_s16x2(dg, E[r], F);
      hd = Hin[r];  // ping-pong buffers: no register moves for the diagonal
      Hl[r] = h;
      const uint32_t t = __vadd2(h, nGsGe);                              // H - Gs - Ge
      E[r] = __viaddmax_s16x2_relu(E[r], nGe, t);                        // Eq. (3)
      F = __viaddmax_s16x2_relu(F, nGe, t);                              // Eq. (4)
      if (r & 1) best = __vimax3_s16x2(best, hprev, dg);
      else hprev = dg;
    }
  }
  Hio = Hl[R - 1];
  Fio = F;
}

// Query-pair variant (two QUERIES per register, one DB sequence): the profile
// already holds (S[qA_i][a], S[qB_i][a]) as s16x2 words, 4 rows per 16-byte
// load, so no PRMT is needed: 5.5 DPX lane-ops per cell pair, of which the
// VIADD.16x2 runs on the FMA pipe (4.5 on the ALU pipe).
template <int R>
__device__ __forceinline__ void gotoh_column_q2(const uint32_t (&Hin)[R], uint32_t (&Hl)[R], uint32_t (&E)[R],
                                                uint32_t& best,
                                                uint32_t& hdiag, const uint8_t* __restrict__ pa, uint32_t& Hio,
                                                uint32_t& Fio, uint32_t nGe, uint32_t nGsGe) {
  static_assert(R % 4 == 0, "R must be a multiple of 4");
  uint32_t hd = hdiag;
  hdiag = Hio;
  uint32_t F = Fio;
  uint32_t hprev = 0;
#pragma unroll
  for (int u = 0; u < R / 4; ++u) {
    const uint4 w = *reinterpret_cast<const uint4*>(pa + u * 16);
    const uint32_t sv[4] = {w.x, w.y, w.z, w.w};
#pragma unroll
    for (int j = 0; j < 4; ++j) {
      const int r = u * 4 + j;
      const uint32_t dg = __vadd2(hd, sv[j]);                              // FMA pipe
      const uint32_t h = __vimax3_s16x2(dg, E[r], F);                       // Eq. (2)
      hd = Hin[r];
      Hl[r] = h;
      const uint32_t t = __vadd2(h, nGsGe);
      E[r] = __viaddmax_s16x2_relu(E[r], nGe, t);                          // Eq. (3)
      F = __viaddmax_s16x2_relu(F, nGe, t);                                // Eq. (4)
      if (r & 1) best = __vimax3_s16x2(best, hprev, dg);                   // max D = max H
      else hprev = dg;
    }
  }
  Hio = Hl[R - 1];
  Fio = F;
}

// Lane block of the query-pair profile: R 4-byte rows, rounded to an odd number
// of 16-byte units (bank-conflict-free LDS.128 across the 8 lanes of a phase).
__host__ __device__ constexpr int lane_block_bytes_q2(int R) { return (((R / 4) | 1) * 16); }

}  // namespace swdual
