// Pipe attribution probe for the Gotoh cell-pair instruction mix on sm_100a.
// Each kernel runs NACC independent chains; per iteration it issues a fixed
// mix. If two opcodes share a pipe, their mix rate equals the sum of their
// individual costs; if not, they overlap. Reports instructions/clk/SM.
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

constexpr int NACC = 8;
constexpr int ITERS = 2048;

__device__ __forceinline__ uint32_t prmt(uint32_t a, uint32_t b, uint32_t sel) {
  uint32_t d;
  asm volatile("prmt.b32 %0, %1, %2, %3;" : "=r"(d) : "r"(a), "r"(b), "r"(sel));
  return d;
}

template <int MIX>
__global__ void k_mix(uint32_t* out, uint32_t seed) {
  uint32_t a[NACC], b[NACC], c[NACC];
  const uint32_t k1 = seed * 0x9E3779B9u, k2 = seed ^ 0x55aa55aau;
#pragma unroll
  for (int i = 0; i < NACC; ++i) { a[i] = seed + i; b[i] = seed * 3 + i; c[i] = seed * 7 + i; }
  for (int it = 0; it < ITERS; ++it) {
#pragma unroll
    for (int i = 0; i < NACC; ++i) {
      if constexpr (MIX == 0) {          // 1 VIADDMNMX
        a[i] = __viaddmax_s16x2_relu(a[i], k1, b[i]);
      } else if constexpr (MIX == 1) {   // 1 VIADD.16x2
        a[i] = __vadd2(a[i], b[i]);
      } else if constexpr (MIX == 2) {   // 1 PRMT
        a[i] = prmt(a[i], b[i], 0xC480);
      } else if constexpr (MIX == 3) {   // VIADDMNMX + VIADD.16x2 (independent)
        a[i] = __viaddmax_s16x2_relu(a[i], k1, c[i]);
        b[i] = __vadd2(b[i], k2);
      } else if constexpr (MIX == 4) {   // VIADDMNMX + PRMT (independent)
        a[i] = __viaddmax_s16x2_relu(a[i], k1, c[i]);
        b[i] = prmt(b[i], c[i], 0xC480);
      } else if constexpr (MIX == 5) {   // VIADDMNMX + IMAD
        a[i] = __viaddmax_s16x2_relu(a[i], k1, c[i]);
        asm volatile("mad.lo.u32 %0, %0, %1, %2;" : "+r"(b[i]) : "r"(k2), "r"(c[i]));
      } else if constexpr (MIX == 6) {   // VIADDMNMX + VIMNMX (s16x2 2-input max)
        a[i] = __viaddmax_s16x2_relu(a[i], k1, c[i]);
        asm volatile("max.s16x2 %0, %0, %1;" : "+r"(b[i]) : "r"(c[i]));
        c[i] += 0x00010001u;
      } else if constexpr (MIX == 8) {   // 1 HMNMX2 (max.f16x2)
        asm volatile("max.f16x2 %0, %0, %1;" : "+r"(a[i]) : "r"(c[i]));
        c[i] += 0x00010001u;
      } else if constexpr (MIX == 9) {   // VIADDMNMX + HMNMX2 (independent)
        a[i] = __viaddmax_s16x2_relu(a[i], k1, c[i]);
        asm volatile("max.f16x2 %0, %0, %1;" : "+r"(b[i]) : "r"(c[i]));
      } else if constexpr (MIX == 10) {  // VIADD.16x2 + HMNMX2 (independent)
        a[i] = __vadd2(a[i], k1);
        asm volatile("max.f16x2 %0, %0, %1;" : "+r"(b[i]) : "r"(c[i]));
      } else if constexpr (MIX == 11) {  // 2 VIADDMNMX + VIADD.16x2 + HMNMX2
        a[i] = __viaddmax_s16x2_relu(a[i], k1, c[i]);
        c[i] = __viaddmax_s16x2_relu(c[i], k2, a[i]);
        asm volatile("add.s16x2 %0, %0, %1;" : "+r"(b[i]) : "r"(k1));
        asm volatile("max.f16x2 %0, %0, %1;" : "+r"(b[i]) : "r"(a[i]));
      } else if constexpr (MIX == 7) {   // VIADDMNMX + SHFL-free SEL/LOP3
        a[i] = __viaddmax_s16x2_relu(a[i], k1, c[i]);
        asm volatile("lop3.b32 %0, %0, %1, %2, 0x96;" : "+r"(b[i]) : "r"(k2), "r"(c[i]));
        asm volatile("lop3.b32 %0, %0, %1, %2, 0x6a;" : "+r"(c[i]) : "r"(k1), "r"(b[i]));
      }
    }
  }
  uint32_t r = 0;
#pragma unroll
  for (int i = 0; i < NACC; ++i) r ^= a[i] ^ b[i] ^ c[i];
  if (r == 0x12345678u) out[blockIdx.x] = r;
}

template <int MIX>
static void run(const char* name, int instr_per_inner, int sms, uint32_t* d) {
  const int block = 256, grid = sms * 8;
  cudaEvent_t e0, e1;
  cudaEventCreate(&e0);
  cudaEventCreate(&e1);
  k_mix<MIX><<<grid, block>>>(d, 1);
  cudaEventRecord(e0);
  for (int i = 0; i < 5; ++i) k_mix<MIX><<<grid, block>>>(d, 2 + i);
  cudaEventRecord(e1);
  cudaEventSynchronize(e1);
  float ms;
  cudaEventElapsedTime(&ms, e0, e1);
  ms /= 5;
  const double warp_instr = double(grid) * (block / 32) * ITERS * NACC * instr_per_inner;
  // instructions per SM per ns; divide by clock (GHz) offline
  printf("{\"mix\":\"%s\",\"ms\":%.4f,\"warp_instr_per_sm_per_ns\":%.3f}\n", name, ms,
         warp_instr / sms / (ms * 1e6));
}

int main() {
  int sms = 0;
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  uint32_t* d;
  cudaMalloc(&d, 1 << 20);
  run<0>("viaddmnmx", 1, sms, d);
  run<1>("viadd16x2", 1, sms, d);
  run<2>("prmt", 1, sms, d);
  run<3>("viaddmnmx+viadd16x2", 2, sms, d);
  run<4>("viaddmnmx+prmt", 2, sms, d);
  run<5>("viaddmnmx+imad", 2, sms, d);
  run<6>("viaddmnmx+vimnmx+iadd", 3, sms, d);
  run<7>("viaddmnmx+lop3x2", 3, sms, d);
  run<8>("hmnmx2+iadd", 2, sms, d);
  run<9>("viaddmnmx+hmnmx2", 2, sms, d);
  run<10>("viadd16x2+hmnmx2", 2, sms, d);
  run<11>("2viaddmnmx+viadd16x2+hmnmx2", 4, sms, d);
  return 0;
}
