// Microbenchmark: the HBM ceiling of a radix-partition pass's access pattern on B200, with no
// shared-memory work at all (destinations are computed arithmetically).
//   read  : stream 2 x n u32 columns (SoA key + payload), 128-bit loads
//   copy  : read SoA, write the AoS u64 tuples sequentially (a perfect 1-partition pass)
//   runs  : read SoA, write each 8192-tuple tile as F runs of 8192/F tuples, run d of tile t to
//           region d at offset t * run (F write streams, one run per warp store group) -- the
//           pattern a pass with fan-out F produces on uniform keys
//   scat  : the same F streams, but element i of a tile goes to stream i % F: every lane of a
//           warp stores to a different stream (no shared-memory shuffle; write combining is
//           left to L2) -- the ceiling of a pass that scatters tuples straight from registers
// n = 2^28 tuples (c3's pass 1: R + S). Prints GB/s of (read + write) bytes per variant.
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o mb_scatter mb_scatter.cu
#include <cstdint>
#include <cstdio>
#include <cuda_runtime.h>

constexpr int NT = 1024, IT = 8, TILE = NT * IT;

__global__ void __launch_bounds__(NT) k_read(const uint4* __restrict__ k, const uint4* __restrict__ p, size_t nv,
                                             uint32_t* sink) {
  uint32_t acc = 0;
  for (size_t i = blockIdx.x * (size_t)NT + threadIdx.x; i < nv; i += (size_t)gridDim.x * NT) {
    const uint4 a = __ldcs(k + i), b = __ldcs(p + i);
    acc ^= a.x ^ a.y ^ a.z ^ a.w ^ b.x ^ b.y ^ b.z ^ b.w;
  }
  if (acc == 0x12345678u) sink[0] = acc;
}

// MODE 0: sequential AoS write; MODE 1: F runs per tile; MODE 2: scattered (element i -> stream i % F)
template <int MODE>
__global__ void __launch_bounds__(NT) k_pass(const uint32_t* __restrict__ keys, const uint32_t* __restrict__ pays,
                                             size_t n, unsigned long long* __restrict__ out, int F) {
  const size_t tiles = n / TILE;
  const int run = TILE / F;
  for (size_t t = blockIdx.x; t < tiles; t += gridDim.x) {
    const uint4* kv = reinterpret_cast<const uint4*>(keys + t * TILE);
    const uint4* pv = reinterpret_cast<const uint4*>(pays + t * TILE);
    #pragma unroll
    for (int j = 0; j < IT / 4; ++j) {
      const uint4 a = __ldcs(kv + j * NT + threadIdx.x), b = __ldcs(pv + j * NT + threadIdx.x);
      const uint32_t ka[4] = {a.x, a.y, a.z, a.w}, pa[4] = {b.x, b.y, b.z, b.w};
      #pragma unroll
      for (int e = 0; e < 4; ++e) {
        // element i of the tile in a 1024-strided layout (as the real pass writes from smem)
        const uint32_t i = (uint32_t)(j * 4 + e) * NT + threadIdx.x;
        const unsigned long long v = (unsigned long long)ka[e] | ((unsigned long long)pa[e] << 32);
        size_t dst;
        if (MODE == 0) dst = t * TILE + i;
        else if (MODE == 1) dst = (size_t)(i / run) * (n / F) + t * run + (i % run);
        else dst = (size_t)(i % F) * (n / F) + t * run + (i / F);
        __stcs(out + dst, v);
      }
    }
  }
}

int main() {
  const size_t n = (size_t)1 << 28;
  uint32_t *k, *p, *sink;
  unsigned long long* out;
  cudaMalloc(&k, n * 4);
  cudaMalloc(&p, n * 4);
  cudaMalloc(&out, n * 8);
  cudaMalloc(&sink, 64);
  cudaMemset(k, 1, n * 4);
  cudaMemset(p, 2, n * 4);
  int sms = 0;
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  cudaEvent_t e0, e1;
  cudaEventCreate(&e0);
  cudaEventCreate(&e1);
  auto time = [&](auto launch, double bytes, const char* name) {
    for (int w = 0; w < 3; ++w) launch();
    cudaEventRecord(e0);
    const int R = 20;
    for (int r = 0; r < R; ++r) launch();
    cudaEventRecord(e1);
    cudaEventSynchronize(e1);
    float ms = 0;
    cudaEventElapsedTime(&ms, e0, e1);
    ms /= R;
    printf("%-28s %8.3f ms  %8.1f GB/s\n", name, ms, bytes / (ms * 1e-3) / 1e9);
  };
  for (int bps : {1, 2}) {
    const int g = sms * bps;
    char nm[64];
    snprintf(nm, sizeof nm, "read (grid %d)", g);
    time([&] { k_read<<<g, NT>>>((const uint4*)k, (const uint4*)p, n / 4, sink); }, 8.0 * n, nm);
    snprintf(nm, sizeof nm, "copy SoA->AoS (grid %d)", g);
    time([&] { k_pass<0><<<g, NT>>>(k, p, n, out, 1); }, 16.0 * n, nm);
    for (int F : {64, 128, 256, 512, 1024}) {
      snprintf(nm, sizeof nm, "runs F=%d run=%d (grid %d)", F, TILE / F, g);
      time([&] { k_pass<1><<<g, NT>>>(k, p, n, out, F); }, 16.0 * n, nm);
    }
    for (int F : {32, 128, 1024, 8192}) {
      snprintf(nm, sizeof nm, "scat F=%d (grid %d)", F, g);
      time([&] { k_pass<2><<<g, NT>>>(k, p, n, out, F); }, 16.0 * n, nm);
    }
  }
  cudaError_t e = cudaDeviceSynchronize();
  printf("status: %s\n", cudaGetErrorString(e));
  return 0;
}
