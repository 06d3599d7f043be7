// Does compute-sanitizer racecheck model mbarrier hand-offs between warps? A correct ping-pong:
// warp 0 writes a shared buffer and arrives on `full`; warp 1 waits on `full`, reads the buffer
// and arrives on `empty`; warp 0 waits on `empty` before writing again (the k_pass_ws stage ring
// in miniature). `racecheck` hazards reported here are false positives of the tool.
//   nvcc -gencode arch=compute_100a,code=sm_100a -o mb_mbar_race mb_mbar_race.cu
//   compute-sanitizer --tool racecheck ./mb_mbar_race
#include <cstdint>
#include <cstdio>

__device__ __forceinline__ uint32_t sa(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
__device__ __forceinline__ void arrive(unsigned long long* b) {
  asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(sa(b)) : "memory");
}
__device__ __forceinline__ void wait(unsigned long long* b, uint32_t par) {
  uint32_t ok = 0;
  while (!ok)
    asm volatile("{\n\t.reg .pred p;\n\tmbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n\tselp.u32 %0, 1, 0, p;\n\t}"
                 : "=r"(ok) : "r"(sa(b)), "r"(par) : "memory");
}

__global__ void k(uint32_t* out) {
  __shared__ uint32_t buf[32];
  __shared__ __align__(8) unsigned long long full, empty;
  if (threadIdx.x == 0) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(sa(&full)) : "memory");
    asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(sa(&empty)) : "memory");
  }
  __syncthreads();
  const int w = threadIdx.x >> 5, l = threadIdx.x & 31;
  uint32_t acc = 0;
  for (int it = 0; it < 8; ++it) {
    if (w == 0) {
      if (it) wait(&empty, (it - 1) & 1);
      buf[l] = it * 32 + l;
      __syncwarp();
      if (l == 0) arrive(&full);
    } else {
      wait(&full, it & 1);
      acc += buf[31 - l];
      __syncwarp();
      if (l == 0) arrive(&empty);
    }
  }
  if (w == 1) out[l] = acc;
}

int main() {
  uint32_t* d;
  cudaMalloc(&d, 128);
  k<<<1, 64>>>(d);
  uint32_t h[32];
  cudaMemcpy(h, d, 128, cudaMemcpyDeviceToHost);
  printf("mbarrier ping-pong: out[0] = %u (expect %u): %s\n", h[0], 8 * 31 + 32 * 28, h[0] == 8 * 31 + 32 * 28 ? "ok" : "WRONG");
  return 0;
}
