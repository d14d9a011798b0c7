// DPX / integer-ALU throughput microbenchmark for sm_100a.
//
// Measures, for each SASS op the Gotoh cell update uses, the chip-wide issue rate in
// lane-ops per SM per clock, plus the full s16x2 Gotoh cell-pair sequence held in
// registers. These numbers fix the denominator of the DPX/ALU cell roofline reported
// by bench.py.
//
// Build: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o dpx_microbench dpx_microbench.cu
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

#define CK(x) do { cudaError_t e_ = (x); if (e_ != cudaSuccess) { \
  fprintf(stderr, "CUDA %s at %s:%d\n", cudaGetErrorString(e_), __FILE__, __LINE__); return 1; } } while (0)

constexpr int NACC = 8;      // independent chains per thread (ILP)
constexpr int ITERS = 4096;

template <int OP>
__device__ __forceinline__ uint32_t op(uint32_t a, uint32_t b, uint32_t c) {
  if constexpr (OP == 0) return __viaddmax_s16x2_relu(a, b, c);   // VIADDMNMX.S16x2.RELU
  if constexpr (OP == 1) return __vimax_s16x2_relu(a, b) ^ c;      // VIMNMX.S16x2 (+LOP3 noise)
  if constexpr (OP == 2) return __vimax3_s16x2(a, b, c);           // VIMNMX3.S16x2
  if constexpr (OP == 3) return __vadd2(a, b) + c;                 // VIADD.16x2 (+IADD)
  if constexpr (OP == 4) return __byte_perm(a, b, 0x5410) ^ c;     // PRMT (+LOP3)
  if constexpr (OP == 5) return a + b + c;                         // IADD3
  if constexpr (OP == 6) return __viaddmax_s32(a, b, c);           // VIADDMNMX (s32)
  // VIMNMX.S16x2 alone.  Two consecutive relu-max with different b fuse into one
  // VIMNMX3 (round-1 probe read 2x the pipe rate), so the second operand here is
  // the running value rotated by PRMT-free means: a - b on the FMA pipe, then max.
  if constexpr (OP == 7) return __vimax_s16x2_relu(a, __vsub2(c, a));
  if constexpr (OP == 8) return __vadd2(a, b);                     // VIADD.16x2 alone
  if constexpr (OP == 9) return __byte_perm(a, b, 0x5410);         // PRMT alone
  return a;
}

template <int OP>
__global__ void k_op(uint32_t* out, uint32_t seed) {
  uint32_t acc[NACC];
  uint32_t b = seed * 0x9E3779B9u + threadIdx.x, c = seed ^ (blockIdx.x * 7919u);
#pragma unroll
  for (int i = 0; i < NACC; ++i) acc[i] = seed + i * 131u + threadIdx.x;
  for (int it = 0; it < ITERS; ++it) {
#pragma unroll
    for (int i = 0; i < NACC; ++i) acc[i] = op<OP>(acc[i], b, c);
    b += 0x00010001u;
  }
  uint32_t r = 0;
#pragma unroll
  for (int i = 0; i < NACC; ++i) r ^= acc[i];
  if (r == 0x12345678u) out[blockIdx.x] = r;
}

// Full Gotoh s16x2 cell-pair update, R rows per thread, register resident.
// Ops per row: VIADDMNMX(Hd,S,max(E,F)) [2], VIADD t [1], E' [1], F' [1], max3 [0.5].
template <int R, bool PERM>
__global__ void k_cell(uint32_t* out, uint32_t seed) {
  uint32_t H[R], E[R], S[R];
  const uint32_t nge = 0xfffefffeu, ngsge = 0xfff4fff4u;
#pragma unroll
  for (int r = 0; r < R; ++r) { H[r] = (seed + r) & 0x00ff00ffu; E[r] = 0; S[r] = ((r * 3 + threadIdx.x) & 7) * 0x00010001u; }
  uint32_t best = 0, hdiag = 0;
  for (int it = 0; it < ITERS / 4; ++it) {
    uint32_t F = 0, hd = hdiag;
#pragma unroll
    for (int r = 0; r < R; r += 2) {
      uint32_t h0 = __viaddmax_s16x2(hd, S[r], __vimax_s16x2_relu(E[r], F));
      uint32_t t0 = __vadd2(h0, ngsge);
      E[r] = __viaddmax_s16x2_relu(E[r], nge, t0);
      F = __viaddmax_s16x2_relu(F, nge, t0);
      hd = H[r]; H[r] = h0;
      uint32_t h1 = __viaddmax_s16x2(hd, S[r + 1], __vimax_s16x2_relu(E[r + 1], F));
      uint32_t t1 = __vadd2(h1, ngsge);
      E[r + 1] = __viaddmax_s16x2_relu(E[r + 1], nge, t1);
      F = __viaddmax_s16x2_relu(F, nge, t1);
      hd = H[r + 1]; H[r + 1] = h1;
      best = __vimax3_s16x2(best, h0, h1);
    }
    hdiag = F ^ it;  // loop-carried, keeps the compiler honest
    if constexpr (PERM) {
#pragma unroll
      for (int r = 0; r < R; ++r) S[r] = __byte_perm(S[r], S[(r + 1) % R], 0x5432);
    }
  }
  if (best == 0x12345678u) out[blockIdx.x] = best;
}

// Same, with the production formulation: D = Hdiag + S on the FMA pipe,
// H = max3(D, E, F), running max over D -> 3.5 ALU ops per cell pair.
template <int R, bool PERM>
__global__ void k_cell2(uint32_t* out, uint32_t seed) {
  uint32_t H[R], E[R], S[R];
  const uint32_t nge = 0xfffefffeu, ngsge = 0xfff4fff4u;
#pragma unroll
  for (int r = 0; r < R; ++r) { H[r] = (seed + r) & 0x00ff00ffu; E[r] = 0; S[r] = ((r * 3 + threadIdx.x) & 7) * 0x00010001u; }
  uint32_t best = 0, hdiag = 0;
  for (int it = 0; it < ITERS / 4; ++it) {
    uint32_t F = 0, hd = hdiag, dprev = 0;
#pragma unroll
    for (int r = 0; r < R; ++r) {
      const uint32_t dg = __vadd2(hd, S[r]);
      const uint32_t h = __vimax3_s16x2(dg, E[r], F);
      const uint32_t t = __vadd2(h, ngsge);
      E[r] = __viaddmax_s16x2_relu(E[r], nge, t);
      F = __viaddmax_s16x2_relu(F, nge, t);
      hd = H[r]; H[r] = h;
      if (r & 1) best = __vimax3_s16x2(best, dprev, dg); else dprev = dg;
    }
    hdiag = F ^ it;
    if constexpr (PERM) {
#pragma unroll
      for (int r = 0; r < R; ++r) S[r] = __byte_perm(S[r], S[(r + 1) % R], 0x5432);
    }
  }
  if (best == 0x12345678u) out[blockIdx.x] = best;
}

// k_cell2 with NCH independent F chains per thread (rows interleaved chain by
// chain, as gotoh_rows_dual does for NCH = 2): how far more ILP per warp lifts
// the latency-bound cell rate at a fixed occupancy.
template <int R, int NCH>
__global__ void k_cellN(uint32_t* out, uint32_t seed) {
  constexpr int RC = R / NCH;
  uint32_t H[R], E[R], S[R];
  const uint32_t nge = 0xfffefffeu, ngsge = 0xfff4fff4u;
#pragma unroll
  for (int r = 0; r < R; ++r) { H[r] = (seed + r) & 0x00ff00ffu; E[r] = 0; S[r] = ((r * 3 + threadIdx.x) & 7) * 0x00010001u; }
  uint32_t best = 0, hdiag = 0;
  for (int it = 0; it < ITERS / 4; ++it) {
    uint32_t F[NCH], hd[NCH], dprev[NCH];
#pragma unroll
    for (int c = 0; c < NCH; ++c) { F[c] = 0; hd[c] = hdiag + c; dprev[c] = 0; }
#pragma unroll
    for (int i = 0; i < RC; ++i) {
#pragma unroll
      for (int c = 0; c < NCH; ++c) {
        const int r = c * RC + i;
        const uint32_t dg = __vadd2(hd[c], S[r]);
        const uint32_t h = __vimax3_s16x2(dg, E[r], F[c]);
        const uint32_t t = __vadd2(h, ngsge);
        E[r] = __viaddmax_s16x2_relu(E[r], nge, t);
        F[c] = __viaddmax_s16x2_relu(F[c], nge, t);
        hd[c] = H[r]; H[r] = h;
        if (i & 1) best = __vimax3_s16x2(best, dprev[c], dg); else dprev[c] = dg;
      }
    }
    uint32_t x = 0;
#pragma unroll
    for (int c = 0; c < NCH; ++c) x ^= F[c];
    hdiag = x ^ it;
  }
  if (best == 0x12345678u) out[blockIdx.x] = best;
}

__global__ void k_clock(unsigned long long* t) {
  unsigned long long c0 = clock64();
  uint32_t x = threadIdx.x;
  for (int i = 0; i < (1 << 22); ++i) x = x * 1664525u + 1013904223u;
  unsigned long long c1 = clock64();
  if (threadIdx.x == 0) t[blockIdx.x] = c1 - c0;
  if (x == 7) t[1] = x;
}

template <typename K>
static float time_kernel(K kern, int grid, int block, uint32_t* d_out) {
  cudaEvent_t a, b;
  cudaEventCreate(&a); cudaEventCreate(&b);
  kern<<<grid, block>>>(d_out, 1u);
  cudaEventRecord(a);
  for (int i = 0; i < 5; ++i) kern<<<grid, block>>>(d_out, 2u + i);
  cudaEventRecord(b);
  cudaEventSynchronize(b);
  float ms = 0; cudaEventElapsedTime(&ms, a, b);
  return ms / 5;
}

int main() {
  int dev = 0; CK(cudaSetDevice(dev));
  cudaDeviceProp p; CK(cudaGetDeviceProperties(&p, dev));
  int sms = p.multiProcessorCount;
  uint32_t* d_out; CK(cudaMalloc(&d_out, 1 << 20));
  unsigned long long* d_t; CK(cudaMalloc(&d_t, 1 << 16));
  // effective SM clock: cycles of a 1-block kernel / event time
  {
    cudaEvent_t a, b; cudaEventCreate(&a); cudaEventCreate(&b);
    k_clock<<<sms, 128>>>(d_t);
    cudaEventRecord(a); k_clock<<<sms, 128>>>(d_t); cudaEventRecord(b); cudaEventSynchronize(b);
    float ms; cudaEventElapsedTime(&ms, a, b);
    unsigned long long cyc; cudaMemcpy(&cyc, d_t, 8, cudaMemcpyDeviceToHost);
    printf("{\"probe\":\"clock\",\"sms\":%d,\"cycles\":%llu,\"ms\":%.4f,\"eff_mhz\":%.1f}\n", sms, cyc, ms, cyc / (ms * 1e3));
  }
  const int block = 256, grid = sms * 8;
  const double lanes = double(grid) * block;
  const char* names[] = {"viaddmax_s16x2_relu", "vimax_s16x2_relu+lop3", "vimax3_s16x2", "vadd2+iadd",
                         "prmt+lop3", "iadd3", "viaddmax_s32", "vimax_s16x2_relu+vsub2(fma)", "vadd2", "prmt"};
  float ms[10];
  ms[0] = time_kernel(k_op<0>, grid, block, d_out);
  ms[1] = time_kernel(k_op<1>, grid, block, d_out);
  ms[2] = time_kernel(k_op<2>, grid, block, d_out);
  ms[3] = time_kernel(k_op<3>, grid, block, d_out);
  ms[4] = time_kernel(k_op<4>, grid, block, d_out);
  ms[5] = time_kernel(k_op<5>, grid, block, d_out);
  ms[6] = time_kernel(k_op<6>, grid, block, d_out);
  ms[7] = time_kernel(k_op<7>, grid, block, d_out);
  ms[8] = time_kernel(k_op<8>, grid, block, d_out);
  ms[9] = time_kernel(k_op<9>, grid, block, d_out);
  for (int i = 0; i < 10; ++i) {
    double ops = lanes * ITERS * NACC;  // one "op" = one source-level call per lane
    printf("{\"probe\":\"%s\",\"ms\":%.4f,\"Glane_ops_per_s\":%.1f}\n", names[i], ms[i], ops / (ms[i] * 1e6));
  }
  for (int g = 1; g <= 8; g *= 2) {
    float mc = time_kernel(k_cell<16, false>, sms * g, block, d_out);
    double cells = double(sms * g) * block * (ITERS / 4) * 16 * 2;  // 16 rows x 2 cells (s16x2)
    printf("{\"probe\":\"gotoh_cellpair_R16_noperm\",\"blocks_per_sm\":%d,\"ms\":%.4f,\"GCUPS\":%.1f}\n", g, mc, cells / (mc * 1e6));
    mc = time_kernel(k_cell<16, true>, sms * g, block, d_out);
    printf("{\"probe\":\"gotoh_cellpair_R16_perm\",\"blocks_per_sm\":%d,\"ms\":%.4f,\"GCUPS\":%.1f}\n", g, mc, cells / (mc * 1e6));
    mc = time_kernel(k_cell<32, false>, sms * g, block, d_out);
    cells = double(sms * g) * block * (ITERS / 4) * 32 * 2;
    printf("{\"probe\":\"gotoh_cellpair_R32_noperm\",\"blocks_per_sm\":%d,\"ms\":%.4f,\"GCUPS\":%.1f}\n", g, mc, cells / (mc * 1e6));
  }
  for (int g = 1; g <= 4; g *= 2) {
    float mc = time_kernel(k_cell2<24, false>, sms * g, block, d_out);
    double cells = double(sms * g) * block * (ITERS / 4) * 24 * 2;
    printf("{\"probe\":\"gotoh_cellpair_D_max3_R24\",\"blocks_per_sm\":%d,\"ms\":%.4f,\"GCUPS\":%.1f}\n", g, mc, cells / (mc * 1e6));
  }
  for (int g = 1; g <= 4; g *= 2) {
    const double cells = double(sms * g) * block * (ITERS / 4) * 24 * 2;
    float mc = time_kernel(k_cellN<24, 1>, sms * g, block, d_out);
    printf("{\"probe\":\"gotoh_cellpair_R24_chains1\",\"blocks_per_sm\":%d,\"ms\":%.4f,\"GCUPS\":%.1f}\n", g, mc, cells / (mc * 1e6));
    mc = time_kernel(k_cellN<24, 2>, sms * g, block, d_out);
    printf("{\"probe\":\"gotoh_cellpair_R24_chains2\",\"blocks_per_sm\":%d,\"ms\":%.4f,\"GCUPS\":%.1f}\n", g, mc, cells / (mc * 1e6));
    mc = time_kernel(k_cellN<24, 3>, sms * g, block, d_out);
    printf("{\"probe\":\"gotoh_cellpair_R24_chains3\",\"blocks_per_sm\":%d,\"ms\":%.4f,\"GCUPS\":%.1f}\n", g, mc, cells / (mc * 1e6));
    mc = time_kernel(k_cellN<24, 4>, sms * g, block, d_out);
    printf("{\"probe\":\"gotoh_cellpair_R24_chains4\",\"blocks_per_sm\":%d,\"ms\":%.4f,\"GCUPS\":%.1f}\n", g, mc, cells / (mc * 1e6));
  }
  CK(cudaGetLastError());
  return 0;
}
