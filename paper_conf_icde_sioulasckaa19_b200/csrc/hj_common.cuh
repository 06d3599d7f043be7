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
// h ^ (h >> lg) ^ (h >> 2lg) ^ (h >> 3lg), shifts clamped at 32 (funnel shift, no branches)
__device__ __forceinline__ uint32_t slot_fold(uint32_t h, const SlotHash& H) {
  const uint32_t r = h ^ __funnelshift_rc(h, 0u, H.lg) ^ __funnelshift_rc(h, 0u, 2 * H.lg) ^
                     __funnelshift_rc(h, 0u, 3 * H.lg);
  return r & ((1u << H.lg) - 1);
}
__device__ __forceinline__ uint32_t slot_of(uint32_t key, const SlotHash& H) { return slot_fold(key >> H.B, H); }
// two-term fold, used when the key bits above B fit in 2 lg bits (H.nfold <= 1, e.g. every 4-byte
// config of BASELINE.json): 3 instructions instead of 6 per lookup
__device__ __forceinline__ uint32_t slot_of2(uint32_t key, const SlotHash& H) {
  const uint32_t h = key >> H.B;
  return (h ^ (h >> H.lg)) & ((1u << H.lg) - 1);
}
// 64-bit keys: the bits above B folded to 32 by a multiply-xor, then one xor-shift (6 instructions
// instead of 10; any hash gives the same join, chains always compare full keys)
__device__ __forceinline__ uint32_t slot_of2(uint64_t key, const SlotHash& H) {
  const uint64_t h64 = key >> H.B;
  const uint32_t h = (uint32_t)h64 ^ ((uint32_t)(h64 >> 32) * 0x9E3779B1u);
  return (h ^ (h >> H.lg)) & ((1u << H.lg) - 1);
}
template <bool F2, typename K>
__device__ __forceinline__ uint32_t slot_for(K key, const SlotHash& H) {
  if constexpr (F2) return slot_of2(key, H);
  else return slot_of(key, H);
}
__device__ __forceinline__ uint32_t slot_of(uint64_t key, const SlotHash& H) {
  const uint64_t h64 = key >> H.B;
  return slot_fold((uint32_t)h64 ^ ((uint32_t)(h64 >> 32) * 0x9E3779B1u), H);
}

// ---- TMA 1-D bulk copies + mbarriers (sm_90+/sm_100a PTX) ---------------------------------
__device__ __forceinline__ uint32_t smem_u32(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
__device__ __forceinline__ void mbar_init(unsigned long long* bar, uint32_t count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count) : "memory");
}
__device__ __forceinline__ void fence_mbar_init() { asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory"); }
__device__ __forceinline__ void fence_proxy_async() { asm volatile("fence.proxy.async.shared::cta;" ::: "memory"); }
__device__ __forceinline__ void mbar_arrive_expect_tx(unsigned long long* bar, uint32_t bytes) {
  asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes) : "memory");
}
// global -> shared bulk copy; dst, src 16-byte aligned, bytes a multiple of 16
__device__ __forceinline__ void bulk_g2s(void* dst, const void* src, uint32_t bytes, unsigned long long* bar) {
  asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
                   smem_u32(dst)),
               "l"(src), "r"(bytes), "r"(smem_u32(bar))
               : "memory");
}
// TMA prefetch of [src, src + bytes) into L2 (bytes a multiple of 16, src 16-byte aligned)
__device__ __forceinline__ void bulk_prefetch_l2(const void* src, uint32_t bytes) {
  asm volatile("cp.async.bulk.prefetch.L2.global [%0], %1;" ::"l"(src), "r"(bytes) : "memory");
}
__device__ __forceinline__ bool mbar_try_wait(unsigned long long* bar, uint32_t parity) {
  uint32_t ok;
  asm volatile(
      "{\n\t.reg .pred p;\n\tmbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n\tselp.u32 %0, 1, 0, p;\n\t}"
      : "=r"(ok)
      : "r"(smem_u32(bar)), "r"(parity)
      : "memory");
  return ok != 0;
}
__device__ __forceinline__ void mbar_wait(unsigned long long* bar, uint32_t parity) {
  while (!mbar_try_wait(bar, parity)) {
  }
}

// %globaltimer (ns): watchdog deadlines of the exchange's device-side waits
__device__ __forceinline__ unsigned long long global_ns() {
  unsigned long long t;
  asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
  return t;
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

// M independent 64-bit exclusive scans in one pass (one pair of barriers instead of M): v[m] ->
// exclusive prefix of v[m] over the block, total[m] = block sum. tmp: >= M * (NT / 32 + 1).
template <int NT, int M>
__device__ __forceinline__ void block_exclusive_scan64xM(unsigned long long (&v)[M], unsigned long long* tmp,
                                                         unsigned long long (&total)[M]) {
  constexpr int NW = NT / 32;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  unsigned long long x[M];
  #pragma unroll
  for (int m = 0; m < M; ++m) {
    x[m] = v[m];
    #pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      unsigned long long y = __shfl_up_sync(0xffffffffu, x[m], o);
      if (lane >= o) x[m] += y;
    }
    if (lane == 31) tmp[m * (NW + 1) + warp] = x[m];
  }
  __syncthreads();
  if (warp < M) {  // warp m scans the warp totals of value m
    unsigned long long* t = tmp + warp * (NW + 1);
    unsigned long long w = (lane < NW) ? t[lane] : 0ull;
    unsigned long long s = w;
    #pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      unsigned long long y = __shfl_up_sync(0xffffffffu, s, o);
      if (lane >= o) s += y;
    }
    if (lane < NW) t[lane] = s - w;
    if (lane == NW - 1) t[NW] = s;
  }
  __syncthreads();
  #pragma unroll
  for (int m = 0; m < M; ++m) {
    v[m] = tmp[m * (NW + 1) + warp] + x[m] - v[m];
    total[m] = tmp[m * (NW + 1) + NW];
  }
  __syncthreads();
}

// Programmatic dependent launch (HJ_OPT_PDL): a kernel launched with programmatic stream
// serialization may start while its predecessor's last blocks still run; it waits here, before
// its first read of anything the predecessor wrote. A no-op for a normal launch.
__device__ __forceinline__ void pdl_wait() { asm volatile("griddepcontrol.wait;" ::: "memory"); }

}  // namespace hj
