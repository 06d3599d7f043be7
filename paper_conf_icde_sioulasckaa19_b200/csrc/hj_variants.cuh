// hj_variants.cuh -- the paper's comparator join algorithms, selectable with
// HJ_OPT_JOIN_ALGO; results are identical to the default path.
//
//   k_join_nlj   co-partition nested-loop join with warp ballots (§III-B, Listing 1,
//                P:319-359): after partitioning, the R chunk sits in shared memory; each warp
//                holds 32 S tuples (one per lane) and scans R 32 values at a time, each lane
//                reading one; for every key bit NOT fixed by the partitioning (bits >= B,
//                P:353-355) a ballot broadcasts the 32 R bits and each lane narrows its match
//                mask (Listing 1 lines 6-9). Matches are then read off the mask (line 10).
//   k_np_build / k_np_probe
//                non-partitioned GPU hash join with a device-memory chained table (the paper's
//                "GPU Non-partitioned" baseline of Fig. 8): build pushes every R row
//                onto its slot's chain with atomicExch; each probe walks its chain in global
//                memory (3-4 random accesses per probe).
#pragma once
#include "hj_common.cuh"
#include "hj_join.cuh"
#include "hj_plan.cuh"

namespace hj {

// ---- output helpers shared by the comparators --------------------------------------------------
// Materialize one warp-step's matches: every lane has m (0/1 here) pairs; one global atomic per
// warp step reserves the range (comparators only: simple, not contention-optimised).
template <typename K>
__device__ __forceinline__ void warp_emit(const Plan& P, bool has, K rpay, K spay) {
  const uint32_t b = __ballot_sync(0xffffffffu, has);
  if (!b) return;
  const int lane = threadIdx.x & 31;
  unsigned long long base = 0;
  if (lane == __ffs(b) - 1) base = atomicAdd(&P.results[RES_CURSOR], (unsigned long long)__popc(b));
  base = __shfl_sync(0xffffffffu, base, __ffs(b) - 1);
  if (has) {
    const unsigned long long pos = base + __popc(b & lanemask_lt());
    if (pos < P.out_cap) {
      ((K*)P.out_r)[pos] = rpay;
      ((K*)P.out_s)[pos] = spay;
    }
  }
}

template <int NT>
__device__ __forceinline__ void block_commit(const Plan& P, unsigned long long cnt, unsigned long long chk) {
  __shared__ unsigned long long s_red[2][NT / 32];
  #pragma unroll
  for (int o = 16; o; o >>= 1) {
    cnt += __shfl_xor_sync(0xffffffffu, cnt, o);
    chk += __shfl_xor_sync(0xffffffffu, chk, o);
  }
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  if (lane == 0) {
    s_red[0][warp] = cnt;
    s_red[1][warp] = chk;
  }
  __syncthreads();
  if (threadIdx.x == 0) {
    unsigned long long c = 0, h = 0;
    for (int w = 0; w < NT / 32; ++w) {
      c += s_red[0][w];
      h += s_red[1][w];
    }
    if (c) {
      atomicAdd(&P.results[RES_MATCHES], c);
      atomicAdd(&P.results[RES_CHECKSUM], h);
    }
  }
}

// ---- ballot nested-loop join over the planner's work items -----------------------------------
template <typename K, int NT, bool MAT>
__global__ void __launch_bounds__(NT) k_join_nlj(Plan P) {
  using TT = Tup<K>;
  using T = typename TT::T;
  constexpr int KB = 8 * sizeof(K);
  extern __shared__ __align__(16) unsigned char s_raw[];
  K* s_rk = reinterpret_cast<K*>(s_raw);  // CR keys
  K* s_rp = s_rk + P.CR;                  // CR payloads
  __shared__ JoinJob s_job;
  const uint32_t total_items = P.ist[1u << P.B];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  unsigned long long my_cnt = 0, my_chk = 0;
  for (;;) {
    if (threadIdx.x == 0) s_job = claim_job<T>(P, total_items);
    __syncthreads();
    const JoinJob job = s_job;
    if (job.item >= total_items) break;
    const T* rsrc = (const T*)P.rel[0].t2 + job.rb;
    for (uint32_t i = threadIdx.x; i < job.nr; i += NT) {
      const T t = rsrc[i];
      s_rk[i] = TT::key(t);
      s_rp[i] = TT::pay(t);
    }
    __syncthreads();
    const T* ssrc = (const T*)P.rel[1].t2;
    for (unsigned long long base = job.sb + (unsigned long long)warp * 32; base < job.se;
         base += (unsigned long long)NT) {
      const unsigned long long s = base + lane;
      const bool active = s < job.se;
      K sk = 0, sp = 0;
      if (active) {
        const T t = ssrc[s];
        sk = TT::key(t);
        sp = TT::pay(t);
      }
      for (uint32_t off = 0; off < job.nr; off += 32) {        // Listing 1 line 3
        const uint32_t l = off + lane;
        const K rk = l < job.nr ? s_rk[l] : K(0);               // line 4
        uint32_t mask = __ballot_sync(0xffffffffu, l < job.nr);  // line 5 (~0 over valid R lanes)
        for (int bit = P.B; bit < KB; ++bit) {                    // line 6: bits not fixed by partitioning
          const uint32_t vote = __ballot_sync(0xffffffffu, (rk >> bit) & 1);  // lines 7-8
          mask &= ((sk >> bit) & 1) ? vote : ~vote;                          // line 9
        }
        if (!active) mask = 0;
        // line 10: matches are the set bits; read each matching lane's payload by shuffle
        if (__any_sync(0xffffffffu, mask != 0)) {
          const K rp = l < job.nr ? s_rp[l] : K(0);
          for (int j = 0; j < 32; ++j) {
            const K rpj = __shfl_sync(0xffffffffu, rp, j);
            const bool hit = (mask >> j) & 1;
            if (MAT) warp_emit<K>(P, hit, rpj, sp);
            if (hit) {
              ++my_cnt;
              if (!MAT || P.mat_chk) my_chk += pair_sig((uint64_t)rpj, (uint64_t)sp);
            }
          }
        }
      }
    }
    __syncthreads();
  }
  block_commit<NT>(P, my_cnt, my_chk);
}

// ---- non-partitioned hash join (device-memory chained table) ----------------------------------
__device__ __forceinline__ uint32_t np_slot(uint32_t k, int lg) { return (k * 0x9E3779B1u) >> (32 - lg); }
__device__ __forceinline__ uint32_t np_slot(uint64_t k, int lg) {
  return (uint32_t)((k * 0x9E3779B97F4A7C15ull) >> (64 - lg));
}

template <typename K>
__global__ void __launch_bounds__(512) k_np_build(const K* __restrict__ keys, unsigned long long n, uint32_t* heads,
                                                  uint32_t* next, int lg) {
  for (unsigned long long i = blockIdx.x * 512ull + threadIdx.x; i < n; i += (unsigned long long)gridDim.x * 512)
    next[i] = atomicExch(&heads[np_slot(keys[i], lg)], (uint32_t)i);
}

template <typename K, bool MAT>
__global__ void __launch_bounds__(512) k_np_probe(Plan P, const K* __restrict__ rk, const K* __restrict__ rp,
                                                  const K* __restrict__ sk, const K* __restrict__ sp,
                                                  unsigned long long nS, const uint32_t* __restrict__ heads,
                                                  const uint32_t* __restrict__ next, int lg) {
  unsigned long long my_cnt = 0, my_chk = 0;
  const unsigned long long stride = (unsigned long long)gridDim.x * 512;
  // trip count uniform across the warp so warp_emit's ballots see every lane
  for (unsigned long long b = blockIdx.x * 512ull + (threadIdx.x & ~31u); b < nS; b += stride) {
    const unsigned long long j = b + (threadIdx.x & 31);
    const bool active = j < nS;
    K key = 0, pay = 0;
    uint32_t i = 0xffffffffu;
    if (active) {
      key = sk[j];
      pay = sp[j];
      i = heads[np_slot(key, lg)];
    }
    while (__any_sync(0xffffffffu, i != 0xffffffffu)) {
      const bool hit = i != 0xffffffffu && rk[i] == key;
      const K r = hit ? rp[i] : K(0);
      if (MAT) warp_emit<K>(P, hit, r, pay);
      if (hit) {
        ++my_cnt;
        if (!MAT || P.mat_chk) my_chk += pair_sig((uint64_t)r, (uint64_t)pay);
      }
      if (i != 0xffffffffu) i = next[i];
    }
  }
  block_commit<512>(P, my_cnt, my_chk);
}

}  // namespace hj
