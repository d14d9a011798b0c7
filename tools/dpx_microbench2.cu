// Cell-update ceiling vs (rows per lane, independent chains, CTA shape) on sm_100a.
//
// Round-2 design probe for the inter-task kernel (DESIGN.md "Where the remaining
// third goes"): the s16x2 Gotoh update in the production form (D = Hdiag + S on
// the FMA pipe, H = VIMNMX3(D, E, F), E'/F' = VIADDMNMX.RELU, running max over D
// every two rows = 3.5 ALU-pipe ops per cell pair), register resident, with
// NCH independent F chains of R / NCH rows per lane.  Variants add what the real
// kernel does per column: profile rows loaded from shared memory (LDS.128 per 4
// rows, letter changing every column) and the per-column lane exchange (3 SHFL +
// 3 SEL).  Kernels run ~5-20 ms so launch and ramp do not distort the rate.
//
// Build: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o dpx_microbench2 dpx_microbench2.cu
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

#define CK(x) do { cudaError_t e_ = (x); if (e_ != cudaSuccess) { \
  fprintf(stderr, "CUDA %s at %s:%d\n", cudaGetErrorString(e_), __FILE__, __LINE__); return 1; } } while (0)

constexpr int COLS = 8192;  // columns per thread

__device__ __forceinline__ uint4 lds128(uint32_t a) {
  uint4 v;
  asm volatile("ld.shared.v4.u32 {%0, %1, %2, %3}, [%4];" : "=r"(v.x), "=r"(v.y), "=r"(v.z), "=r"(v.w) : "r"(a));
  return v;
}

// LDS: 0 = S in registers, 1 = S rows from shared memory per column (letter varies).
// XCH: per-column lane exchange (shuffles of the chain-0 inputs + lane-0 selects).
template <int R, int NCH, int LDS, int XCH>
__global__ void k_cell(uint32_t* out, uint32_t seed, int cols) {
  constexpr int RC = R / NCH;
  static_assert(!LDS || RC % 4 == 0, "4-row units");
  __shared__ __align__(16) uint32_t prof[16 * 8 * (R + 4)];  // [letter][lane % 8][row] (padded lane block)
  for (int i = threadIdx.x; i < 16 * 8 * (R + 4); i += blockDim.x) prof[i] = (i * 2654435761u) & 0x00070007u;
  __syncthreads();
  const uint32_t sbase = static_cast<uint32_t>(__cvta_generic_to_shared(prof));
  const int lane = threadIdx.x & 31;
  const uint32_t laneoff = (lane & 7) * (R + 4) * 4;
  uint32_t H[R], E[R], S[R];
  const uint32_t nge = 0xfffefffeu, ngsge = 0xfff4fff4u;
#pragma unroll
  for (int r = 0; r < R; ++r) { H[r] = (seed + r) & 0x00ff00ffu; E[r] = 0; S[r] = ((r * 3 + threadIdx.x) & 7) * 0x00010001u; }
  uint32_t best = 0, hin = 0, fin = 0, code = seed & 15;
  uint32_t hd[NCH], F[NCH];
#pragma unroll
  for (int c = 0; c < NCH; ++c) { hd[c] = c; F[c] = 0; }
  for (int t = 0; t < cols; ++t) {
    if constexpr (XCH) {
      uint32_t rH = __shfl_up_sync(0xffffffffu, H[R - 1], 1, 4);
      uint32_t rF = __shfl_up_sync(0xffffffffu, F[NCH - 1], 1, 4);
      uint32_t rC = __shfl_up_sync(0xffffffffu, code, 1, 4);
      const bool lead = (lane & 3) == 0;
      rH = lead ? hin : rH;
      rF = lead ? fin : rF;
      rC = lead ? ((t * 7 + 3) & 15) : rC;
      hin = rH ^ t;
      fin = rF;
      code = rC;
      F[0] = rF & 0x7fff7fffu;
      hd[0] = rH & 0x7fff7fffu;
    } else {
      code = (code * 5 + 1) & 15;
    }
#pragma unroll
    for (int c = 0; c < NCH; ++c) {
      uint32_t dprev = 0;
#pragma unroll
      for (int i = 0; i < RC; ++i) {
        const int r = c * RC + i;
        if constexpr (LDS) {
          if (i % 4 == 0) {
            const uint4 w = lds128(sbase + ((code + c) & 15) * (8 * (R + 4) * 4) + laneoff + i * 4);
            S[r] = w.x; S[r + 1] = w.y; S[r + 2] = w.z; S[r + 3] = w.w;
          }
        }
        const uint32_t dg = __vadd2(hd[c], S[r]);
        const uint32_t h = __vimax3_s16x2(dg, E[r], F[c]);
        const uint32_t tt = __vadd2(h, ngsge);
        E[r] = __viaddmax_s16x2_relu(E[r], nge, tt);
        F[c] = __viaddmax_s16x2_relu(F[c], nge, tt);
        hd[c] = H[r];
        H[r] = h;
        if (i & 1) best = __vimax3_s16x2(best, dprev, dg); else dprev = dg;
      }
    }
    if constexpr (!XCH) {
#pragma unroll
      for (int c = 0; c < NCH; ++c) { hd[c] ^= (t & 1); F[c] = F[c] & 0x7fff7fffu; }
    }
  }
  uint32_t x = best;
#pragma unroll
  for (int c = 0; c < NCH; ++c) x ^= F[c] ^ hd[c];
  if (x == 0x12345678u) out[blockIdx.x] = x;
}

template <int R, int NCH, int LDS, int XCH>
static int run(const char* tag, int sms, int threads, int ctas_per_sm, uint32_t* d_out) {
  auto kern = k_cell<R, NCH, LDS, XCH>;
  int nreg = 0;
  cudaFuncAttributes fa;
  if (cudaFuncGetAttributes(&fa, kern) == cudaSuccess) nreg = fa.numRegs;
  int occ = 0;
  CK(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, kern, threads, 0));
  if (occ < ctas_per_sm) {
    printf("{\"probe\":\"%s\",\"R\":%d,\"chains\":%d,\"lds\":%d,\"xch\":%d,\"threads\":%d,\"ctas_per_sm\":%d,"
           "\"regs\":%d,\"skip\":\"occupancy %d\"}\n", tag, R, NCH, LDS, XCH, threads, ctas_per_sm, nreg, occ);
    return 0;
  }
  const int grid = sms * ctas_per_sm;
  const int cols = COLS;
  kern<<<grid, threads>>>(d_out, 1u, cols);
  CK(cudaDeviceSynchronize());
  cudaEvent_t a, b;
  cudaEventCreate(&a); cudaEventCreate(&b);
  cudaEventRecord(a);
  for (int i = 0; i < 3; ++i) kern<<<grid, threads>>>(d_out, 2u + i, cols);
  cudaEventRecord(b);
  CK(cudaEventSynchronize(b));
  float ms = 0; cudaEventElapsedTime(&ms, a, b);
  ms /= 3;
  const double cells = double(grid) * threads * cols * R * 2;
  printf("{\"probe\":\"%s\",\"R\":%d,\"chains\":%d,\"lds\":%d,\"xch\":%d,\"threads\":%d,\"ctas_per_sm\":%d,"
         "\"regs\":%d,\"ms\":%.3f,\"GCUPS\":%.1f}\n", tag, R, NCH, LDS, XCH, threads, ctas_per_sm, nreg, ms,
         cells / (ms * 1e6));
  return 0;
}

int main() {
  CK(cudaSetDevice(0));
  cudaDeviceProp p; CK(cudaGetDeviceProperties(&p, 0));
  const int sms = p.multiProcessorCount;
  uint32_t* d_out; CK(cudaMalloc(&d_out, 1 << 20));
  run<24, 2, 0, 0>("cell", sms, 256, 2, d_out);
  run<24, 2, 1, 0>("cell", sms, 256, 2, d_out);
  run<24, 2, 1, 1>("cell", sms, 256, 2, d_out);
  run<24, 2, 1, 1>("cell", sms, 256, 1, d_out);
  run<24, 3, 0, 0>("cell", sms, 256, 2, d_out);
  run<16, 2, 0, 0>("cell", sms, 256, 3, d_out);
  run<16, 2, 1, 1>("cell", sms, 256, 3, d_out);
  run<16, 2, 1, 1>("cell", sms, 256, 2, d_out);
  run<32, 2, 0, 0>("cell", sms, 256, 2, d_out);
  run<32, 2, 1, 1>("cell", sms, 256, 2, d_out);
  run<32, 4, 1, 1>("cell", sms, 256, 2, d_out);
  run<24, 2, 1, 1>("cell", sms, 512, 1, d_out);
  run<24, 2, 1, 1>("cell", sms, 128, 4, d_out);
  run<48, 4, 1, 1>("cell", sms, 256, 1, d_out);
  run<48, 2, 1, 1>("cell", sms, 256, 1, d_out);
  run<40, 2, 1, 1>("cell", sms, 256, 1, d_out);
  run<32, 2, 1, 0>("cell", sms, 256, 2, d_out);
  run<24, 2, 1, 0>("cell", sms, 384, 1, d_out);
  CK(cudaGetLastError());
  return 0;
}
