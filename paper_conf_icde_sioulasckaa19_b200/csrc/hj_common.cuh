// hj_common.cuh -- tuple layouts, block scans and small device helpers shared by the
// partition and join kernels (sm_100a). Nothing here is shared with oracle/.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

namespace hj {

// ------------------------------------------------------------------------------------------
// AoS tuple layouts written by the partition passes (DESIGN.md §4 "layout in HBM").
//   4/4: one uint64 = key | pay << 32  (8 B, one LDG.64/STS.64 per tuple)
//   8/8: ulonglong2 {key, pay}        (16 B)
// ------------------------------------------------------------------------------------------
template <typename K>
struct Tup;

template <>
struct Tup<uint32_t> {
  using T = unsigned long long;
  using K = uint32_t;
  __device__ __forceinline__ static K key(T t) { return (K)(t & 0xffffffffull); }
  __device__ __forceinline__ static K pay(T t) { return (K)(t >> 32); }
  __device__ __forceinline__ static T make(K k, K p) { return (T)k | ((T)p << 32); }
};

template <>
struct Tup<uint64_t> {
  using T = ulonglong2;
  using K = uint64_t;
  __device__ __forceinline__ static K key(T t) { return t.x; }
  __device__ __forceinline__ static K pay(T t) { return t.y; }
  __device__ __forceinline__ static T make(K k, K p) { return make_ulonglong2(k, p); }
};

// splitmix64 finalizer and the pair signature of the aggregated output (S1).
__device__ __forceinline__ uint64_t fmix64(uint64_t z) {
  z ^= z >> 30;
  z *= 0xBF58476D1CE4E5B9ull;
  z ^= z >> 27;
  z *= 0x94D049BB133111EBull;
  z ^= z >> 31;
  return z;
}
__device__ __forceinline__ uint64_t pair_sig(uint64_t r_pay, uint64_t s_pay) {
  return fmix64(r_pay ^ (s_pay * 0x9E3779B97F4A7C15ull));
}

// In-partition slot hash: the key bits above the B radix bits, xor-folded down to lg_nb bits
// with `nfold` extra terms (host-computed: enough terms to cover every remaining key bit, at
// most 3). For dense keys (c1-c4) (key >> B) < nb, so this is the identity on the remaining
// bits (collision-free chains). Chains always compare full keys, so the hash only affects
// speed, never results.
struct SlotHash {
  int B, lg, nfold;
};
__device__ __forceinline__ uint32_t slot_fold(uint32_t h, const SlotHash& H) {
  uint32_t r = h;
  if (H.nfold >= 1) r ^= h >> H.lg;
  if (H.nfold >= 2) r ^= h >> (2 * H.lg);
  if (H.nfold >= 3) r ^= h >> (3 * H.lg);
  return r & ((1u << H.lg) - 1);
}
__device__ __forceinline__ uint32_t slot_of(uint32_t key, const SlotHash& H) { return slot_fold(key >> H.B, H); }
__device__ __forceinline__ uint32_t slot_of(uint64_t key, const SlotHash& H) {
  const uint64_t h64 = key >> H.B;
  return slot_fold((uint32_t)h64 ^ ((uint32_t)(h64 >> 32) * 0x9E3779B1u), H);
}

__device__ __forceinline__ uint32_t lanemask_lt() {
  uint32_t m;
  asm("mov.u32 %0, %%lanemask_lt;" : "=r"(m));
  return m;
}

// Block-wide exclusive scan of one uint32 per thread. `tmp` needs blockDim/32 + 1 words.
// Returns the exclusive prefix; *total gets the block sum. Contains two __syncthreads.
template <int NT>
__device__ __forceinline__ uint32_t block_exclusive_scan(uint32_t v, uint32_t* tmp, uint32_t* total) {
  static_assert(NT % 32 == 0 && NT <= 1024, "block size");
  constexpr int NW = NT / 32;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  uint32_t x = v;
  #pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    uint32_t y = __shfl_up_sync(0xffffffffu, x, o);
    if (lane >= o) x += y;
  }
  if (lane == 31) tmp[warp] = x;
  __syncthreads();
  if (warp == 0) {
    uint32_t w = (lane < NW) ? tmp[lane] : 0u;
    uint32_t s = w;
    #pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      uint32_t y = __shfl_up_sync(0xffffffffu, s, o);
      if (lane >= o) s += y;
    }
    if (lane < NW) tmp[lane] = s - w;
    if (lane == NW - 1) tmp[NW] = s;
  }
  __syncthreads();
  uint32_t res = tmp[warp] + x - v;
  *total = tmp[NW];
  return res;
}

// 64-bit variant (used by the single-block planner).
template <int NT>
__device__ __forceinline__ unsigned long long block_exclusive_scan64(unsigned long long v, unsigned long long* tmp,
                                                                     unsigned long long* total) {
  constexpr int NW = NT / 32;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  unsigned long long x = v;
  #pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    unsigned long long y = __shfl_up_sync(0xffffffffu, x, o);
    if (lane >= o) x += y;
  }
  if (lane == 31) tmp[warp] = x;
  __syncthreads();
  if (warp == 0) {
    unsigned long long w = (lane < NW) ? tmp[lane] : 0ull;
    unsigned long long s = w;
    #pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      unsigned long long y = __shfl_up_sync(0xffffffffu, s, o);
      if (lane >= o) s += y;
    }
    if (lane < NW) tmp[lane] = s - w;
    if (lane == NW - 1) tmp[NW] = s;
  }
  __syncthreads();
  unsigned long long res = tmp[warp] + x - v;
  *total = tmp[NW];
  __syncthreads();
  return res;
}

}  // namespace hj
