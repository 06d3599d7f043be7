// Microbenchmark: shared-memory pipe cost per warp instruction of the access patterns a
// partition pass uses (1024 threads per block, one block per SM, data in registers).
//   0 ATOMS, digit counters        hist[d], d uniform in [0, 256)
//   1 ATOMS, lane-private (LP)     lc[(d >> 1) * 32 + lane] += 1 << 16 (d & 1)
//   2 ATOMS, lane-distinct fixed   lc[lane]
//   3 ATOMS, one address           hist[0]
//   4 ATOMS, lc[d * 32 + lane]     (unpacked lane-private)
//   5 LDS   random word in 256
//   6 LDS   lane-distinct (bank = lane)
//   7 STS.64 random slot in 7680   (the shuffle)
//   8 STS.64 sequential            (lane-contiguous)
//   9 RED-style ATOMS no return, digit counters
// Prints SM clocks per warp instruction (all 32 warps of the SM issue the pattern).
#include <cstdint>
#include <cstdio>
#include <cuda_runtime.h>

__device__ __forceinline__ uint32_t mix(uint32_t x) {
  x ^= x >> 16; x *= 0x7feb352dU; x ^= x >> 15; x *= 0x846ca68bU; x ^= x >> 16; return x;
}

template <int MODE>
__global__ void __launch_bounds__(1024, 1) k(int iters, uint32_t* sink, long long* clk) {
  extern __shared__ __align__(16) uint32_t sh[];
  const uint32_t lane = threadIdx.x & 31;
  for (int i = threadIdx.x; i < 7680 * 2 + 8192; i += 1024) sh[i] = 0;
  __syncthreads();
  uint32_t acc = 0;
  uint32_t seed = blockIdx.x * 7919u + threadIdx.x * 104729u;
  unsigned long long* s64 = reinterpret_cast<unsigned long long*>(sh);
  const long long t0 = clock64();
  for (int it = 0; it < iters; ++it) {
    const uint32_t h = mix(seed + it * 0x9E3779B9u);
    const uint32_t d = h & 255;
    if (MODE == 0) acc += atomicAdd(&sh[d], 1u);
    if (MODE == 1) acc += atomicAdd(&sh[(d >> 1) * 32 + lane], 1u << ((d & 1) << 4));
    if (MODE == 2) acc += atomicAdd(&sh[lane], 1u);
    if (MODE == 3) acc += atomicAdd(&sh[0], 1u);
    if (MODE == 4) acc += atomicAdd(&sh[(d & 127) * 32 + lane], 1u);
    if (MODE == 5) acc += *(volatile uint32_t*)&sh[d];
    if (MODE == 6) acc += *(volatile uint32_t*)&sh[(d >> 1) * 32 + lane];
    if (MODE == 7) *(volatile unsigned long long*)&s64[h % 7680] = h;
    if (MODE == 8) *(volatile unsigned long long*)&s64[((it * 1024 + threadIdx.x) % 7680)] = h;
    if (MODE == 9) atomicAdd(&sh[d], 1u);
  }
  __syncthreads();
  const long long t1 = clock64();
  if (threadIdx.x == 0) clk[blockIdx.x] = t1 - t0;
  if (acc == 0x12345678u) sink[0] = acc;
}

template <int MODE>
void run(const char* name, int sms, uint32_t* sink, long long* clk) {
  const int iters = 4096;
  const size_t sm = (7680 * 2 + 8192) * 4;
  cudaFuncSetAttribute(k<MODE>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sm);
  k<MODE><<<sms, 1024, sm>>>(iters, sink, clk);
  k<MODE><<<sms, 1024, sm>>>(iters, sink, clk);
  cudaDeviceSynchronize();
  long long h[256];
  cudaMemcpy(h, clk, sms * sizeof(long long), cudaMemcpyDeviceToHost);
  double m = 0;
  for (int i = 0; i < sms; ++i) m += h[i];
  m /= sms;
  // 32 warps x iters warp instructions per SM (plus the hash: ~12 ALU instructions per iteration)
  printf("%-34s %6.2f clk per warp instruction\n", name, m / (32.0 * iters));
}

int main() {
  int sms = 148;
  uint32_t* sink;
  long long* clk;
  cudaMalloc(&sink, 4);
  cudaMalloc(&clk, 256 * sizeof(long long));
  run<0>("ATOMS digit counters (256)", sms, sink, clk);
  run<1>("ATOMS lane-private packed (LP)", sms, sink, clk);
  run<2>("ATOMS lane-distinct fixed", sms, sink, clk);
  run<3>("ATOMS one address", sms, sink, clk);
  run<4>("ATOMS lane-private unpacked", sms, sink, clk);
  run<5>("LDS random word in 256", sms, sink, clk);
  run<6>("LDS lane-distinct banks", sms, sink, clk);
  run<7>("STS.64 random slot in 7680", sms, sink, clk);
  run<8>("STS.64 sequential", sms, sink, clk);
  run<9>("ATOMS no-return digit counters", sms, sink, clk);
  return 0;
}
