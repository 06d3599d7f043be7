// Microbenchmark: cost of the in-tile ranking primitives a radix-partition
// pass can use on sm_100a (data in registers, no HBM traffic).
//   mode 0: smem atomicAdd-with-return on 2^bits block-shared counters
//   mode 1: smem atomicAdd no-return (histogram) on 2^bits counters
//   mode 2: __match_any_sync(digit) + leader RMW on a per-warp histogram
//   mode 3: ballot-based match over `bits` bits + leader RMW per-warp histogram
//   mode 4: smem atomicAdd-with-return on per-warp private counters
// Prints tuples/clk/SM for each mode and bits in {8, 15}.
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

__device__ __forceinline__ uint32_t mix(uint32_t x) {
  x ^= x >> 16; x *= 0x7feb352dU; x ^= x >> 15; x *= 0x846ca68bU; x ^= x >> 16; return x;
}

template <int MODE>
__global__ void __launch_bounds__(256) k_rank(int bits, int iters, int skew, uint32_t* sink) {
  extern __shared__ uint32_t sh[];
  const int nb = 1 << bits;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  uint32_t* hist = sh;  // MODE 0/1: nb; MODE 2/3/4: 8 warps * nb (bits<=8 only)
  int total = (MODE >= 2) ? 8 * nb : nb;
  for (int i = threadIdx.x; i < total; i += blockDim.x) hist[i] = 0;
  __syncthreads();
  uint32_t acc = 0;
  uint32_t seed = blockIdx.x * 7919u + threadIdx.x;
  for (int it = 0; it < iters; ++it) {
    uint32_t h = mix(seed + it * 0x9E3779B9u);
    uint32_t d = h & (nb - 1);
    if (skew && (h >> 28) < 6) d = 5;  // ~37% of tuples on one digit
    if (MODE == 0) {
      acc += atomicAdd(&hist[d], 1u);
    } else if (MODE == 1) {
      atomicAdd(&hist[d], 1u);
    } else if (MODE == 2) {
      uint32_t peers = __match_any_sync(0xffffffffu, d);
      int leader = __ffs(peers) - 1;
      uint32_t* wh = hist + warp * nb;
      uint32_t old = 0;
      if (lane == leader) { old = wh[d]; wh[d] = old + __popc(peers); }
      old = __shfl_sync(0xffffffffu, old, leader);
      acc += old + __popc(peers & ((1u << lane) - 1));
      __syncwarp();
    } else if (MODE == 3) {
      uint32_t peers = 0xffffffffu;
#pragma unroll
      for (int b = 0; b < 8; ++b) {
        uint32_t v = __ballot_sync(0xffffffffu, (d >> b) & 1);
        peers &= ((d >> b) & 1) ? v : ~v;
      }
      int leader = __ffs(peers) - 1;
      uint32_t* wh = hist + warp * nb;
      uint32_t old = 0;
      if (lane == leader) { old = wh[d]; wh[d] = old + __popc(peers); }
      old = __shfl_sync(0xffffffffu, old, leader);
      acc += old + __popc(peers & ((1u << lane) - 1));
      __syncwarp();
    } else {
      acc += atomicAdd(&hist[warp * nb + d], 1u);
    }
  }
  __syncthreads();
  if (acc == 0x12345678u) sink[0] = hist[threadIdx.x];
  if (threadIdx.x == 0) sink[1 + blockIdx.x % 64] = acc + hist[0];
}

template <int MODE>
void run(int bits, int skew, int occ) {
  if (MODE >= 2 && bits > 8) return;
  int nb = 1 << bits;
  size_t smem = (MODE >= 2 ? 8 : 1) * nb * 4;
  cudaFuncSetAttribute(k_rank<MODE>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  uint32_t* sink; cudaMalloc(&sink, 4096);
  int iters = 4096;
  int grid = 148 * occ;
  k_rank<MODE><<<grid, 256, smem>>>(bits, iters, skew, sink);
  cudaEvent_t a, b; cudaEventCreate(&a); cudaEventCreate(&b);
  cudaEventRecord(a);
  k_rank<MODE><<<grid, 256, smem>>>(bits, iters, skew, sink);
  cudaEventRecord(b); cudaEventSynchronize(b);
  float ms; cudaEventElapsedTime(&ms, a, b);
  int clk_khz; cudaDeviceGetAttribute(&clk_khz, cudaDevAttrClockRate, 0);
  double tuples = (double)grid * 256 * iters;
  double gt = tuples / (ms * 1e-3) / 1e9;
  // per-SM per-clock at the max clock (lower bound on tuples/clk)
  double tpc = tuples / (ms * 1e-3) / 148 / (clk_khz * 1e3);
  printf("mode=%d bits=%2d skew=%d occ=%d  %.3f ms  %.1f Gtuples/s  %.3f tuples/clk/SM (at %d MHz) err=%s\n",
         MODE, bits, skew, occ, ms, gt, tpc, clk_khz / 1000, cudaGetErrorString(cudaGetLastError()));
  cudaFree(sink);
}

int main() {
  for (int skew = 0; skew < 2; ++skew)
    for (int occ : {4, 8}) {
      for (int bits : {8, 15}) {
        run<0>(bits, skew, occ);
        run<1>(bits, skew, occ);
        run<2>(bits, skew, occ);
        run<3>(bits, skew, occ);
        run<4>(bits, skew, occ);
      }
    }
  return 0;
}
