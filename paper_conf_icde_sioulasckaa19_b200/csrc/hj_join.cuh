// hj_join.cuh -- steps a6-a8 of the hot path: the co-partition join.
//
// One work item = (co-partition q, R chunk, S chunk) from the planner's list, so long S
// co-partitions are spread over many blocks and R co-partitions larger
// than the shared-memory capacity become hash-based block nested loops.
// Blocks are persistent and take items from a global atomic counter.
//
// Build (Listing 2): the R chunk is copied into shared memory
// (AoS tuples); a chained hash table uses one 32-bit head per slot and 16-bit `next` offsets;
// insertion is wait-free push-front with atomicExch.
// Probe: each S tuple (coalesced loads) hashes to its slot and follows the chain
// comparing keys.
// Output: count + pair checksum aggregated per thread and committed with one 64-bit atomic per
// block; or materialized (see k_join below).
#pragma once
#include "hj_common.cuh"
#include "hj_plan.cuh"

namespace hj {

constexpr uint32_t NIL16 = 0xffffu;

struct JoinJob {
  uint32_t item, nr;
  unsigned long long rb, sb, se;
};

// Claim the next work item and decode it (item -> co-partition q by binary search over the
// planner's item prefix; then the R chunk and S chunk of q it covers). One lane.
__device__ __forceinline__ JoinJob claim_job(const Plan& P, uint32_t total_items) {
  JoinJob j;
  j.item = atomicAdd(&P.counters[CNT_NEXT_ITEM], 1u);
  j.nr = 0;
  j.rb = j.sb = j.se = 0;
  if (j.item < total_items) {
    const uint32_t np = 1u << P.B;
    uint32_t lo = 0, hi = np;  // largest q with ist[q] <= item
    while (hi - lo > 1) {
      const uint32_t mid = (lo + hi) >> 1;
      if (P.ist[mid] <= j.item) lo = mid; else hi = mid;
    }
    const uint32_t q = lo;
    const unsigned long long r0 = P.rel[0].off[q], rn = P.rel[0].off[q + 1] - r0;
    const unsigned long long s0 = P.rel[1].off[q], sn = P.rel[1].off[q + 1] - s0;
    const unsigned long long nsch = (sn + P.CS - 1) / P.CS;
    const unsigned long long loc = j.item - P.ist[q];
    const unsigned long long rc = loc / nsch, sc = loc % nsch;
    j.rb = r0 + rc * P.CR;
    j.nr = (uint32_t)min((unsigned long long)P.CR, rn - rc * P.CR);
    j.sb = s0 + sc * P.CS;
    j.se = j.sb + min((unsigned long long)P.CS, sn - sc * P.CS);
  }
  return j;
}

__device__ __forceinline__ void bar_compute(int nthreads) {  // named barrier 1: compute warps only
  asm volatile("bar.sync 1, %0;" ::"r"(nthreads) : "memory");
}

// Block = NT compute threads + one scheduler warp. The scheduler warp claims and decodes item
// k+1 while the compute warps join item k (it only joins the end-of-item barrier), so the
// dependent global loads of the item lookup never stall the join.
//
// Output of the materialized mode: per probe round every thread knows the match count of each
// of its S tuples (first chain walk, which also keeps the first match's payload); the compute
// warps reserve the round's total with ONE global atomicAdd, then each warp carves its range
// per tuple slot with a shared-memory atomic and lanes write their pairs at warp-contiguous
// positions (coalesced stores). This replaces the paper's per-warp buffer + global atomic per
// flush. Chains are re-walked only for S tuples with more than one match.
template <typename K, int NT, int SPT, bool MAT>
__global__ void __launch_bounds__(NT + 32, 3) k_join(Plan P) {
  using TT = Tup<K>;
  using T = typename TT::T;
  extern __shared__ __align__(16) unsigned char s_raw[];
  const SlotHash H = P.H;
  const uint32_t nb = 1u << H.lg;
  T* s_rt = reinterpret_cast<T*>(s_raw);                        // CR tuples
  uint32_t* s_head = reinterpret_cast<uint32_t*>(s_rt + P.CR);  // nb
  uint16_t* s_next = reinterpret_cast<uint16_t*>(s_head + nb);  // CR
  __shared__ JoinJob s_jobs[2];
  __shared__ unsigned long long s_base;
  __shared__ uint32_t s_wcur;
  __shared__ uint32_t s_wsum[NT / 32];
  __shared__ unsigned long long s_red[2][NT / 32 + 1];

  const uint32_t total_items = P.ist[1u << P.B];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const bool sched = threadIdx.x >= NT;
  K* out_r = (K*)P.out_r;
  K* out_s = (K*)P.out_s;
  const T* ssrc = (const T*)P.rel[1].t2;
  unsigned long long my_cnt = 0, my_chk = 0;

  if (sched && lane == 0) s_jobs[0] = claim_job(P, total_items);
  __syncthreads();

  for (uint32_t it = 0;; ++it) {
    const JoinJob job = s_jobs[it & 1];
    if (job.item >= total_items) break;
    if (sched) {
      if (lane == 0) s_jobs[(it + 1) & 1] = claim_job(P, total_items);
      __syncthreads();  // end-of-item barrier (matches the compute warps' one below)
      continue;
    }

    // ---- issue the first probe round's S loads, then the R chunk (all in flight together) ----
    K sk[SPT], sp[SPT];
    auto load_s = [&](unsigned long long base) {
      #pragma unroll
      for (int j = 0; j < SPT; ++j) {
        const unsigned long long s = base + (unsigned long long)j * NT + threadIdx.x;
        if (s < job.se) {
          const T t = __ldcs(ssrc + s);
          sk[j] = TT::key(t);
          sp[j] = TT::pay(t);
        }
      }
    };
    load_s(job.sb);
    {
      const T* rsrc = (const T*)P.rel[0].t2 + job.rb;
      for (uint32_t i = threadIdx.x; i < nb; i += NT) s_head[i] = NIL16;
      constexpr int U = 4;
      for (uint32_t i = threadIdx.x; i < job.nr; i += U * NT) {
        T v[U];
        #pragma unroll
        for (int u = 0; u < U; ++u)
          if (i + u * NT < job.nr) v[u] = __ldcs(rsrc + i + u * NT);
        #pragma unroll
        for (int u = 0; u < U; ++u)
          if (i + u * NT < job.nr) s_rt[i + u * NT] = v[u];
      }
    }
    bar_compute(NT);
    // ---- build (a6): wait-free push-front insert (Listing 2) ----------------------
    for (uint32_t i = threadIdx.x; i < job.nr; i += NT)
      s_next[i] = (uint16_t)atomicExch(&s_head[slot_of(TT::key(s_rt[i]), H)], i);
    bar_compute(NT);

    // ---- probe (a7) + output (a8), SPT tuples per thread per round --------------------------
    for (unsigned long long base = job.sb; base < job.se; base += (unsigned long long)NT * SPT) {
      if (base != job.sb) load_s(base);
      uint32_t idx[SPT], m[SPT];
      K rfirst[SPT];
      #pragma unroll
      for (int j = 0; j < SPT; ++j) {
        const unsigned long long s = base + (unsigned long long)j * NT + threadIdx.x;
        idx[j] = (s < job.se) ? s_head[slot_of(sk[j], H)] : NIL16;
        m[j] = 0;
      }
      // chains of all SPT tuples advance together (independent shared-memory loads in flight)
      bool live = true;
      while (live) {
        live = false;
        #pragma unroll
        for (int j = 0; j < SPT; ++j) {
          if (idx[j] != NIL16) {
            const T r = s_rt[idx[j]];
            if (TT::key(r) == sk[j]) {
              if (MAT) {
                if (m[j] == 0) rfirst[j] = TT::pay(r);
              } else {
                my_chk += pair_sig((uint64_t)TT::pay(r), (uint64_t)sp[j]);
              }
              ++m[j];
            }
            idx[j] = s_next[idx[j]];
            live |= idx[j] != NIL16;
          }
        }
      }
      uint32_t mt = 0;
      #pragma unroll
      for (int j = 0; j < SPT; ++j) mt += m[j];
      my_cnt += mt;
      if (MAT) {
        const uint32_t wsum = __reduce_add_sync(0xffffffffu, mt);
        if (lane == 0) s_wsum[warp] = wsum;
        bar_compute(NT);
        if (threadIdx.x == 0) {
          uint32_t tot = 0;
          #pragma unroll
          for (int w = 0; w < NT / 32; ++w) tot += s_wsum[w];
          s_base = tot ? atomicAdd(&P.results[RES_CURSOR], (unsigned long long)tot) : 0ull;
          s_wcur = 0;
        }
        bar_compute(NT);
        const unsigned long long gbase = s_base;
        #pragma unroll
        for (int j = 0; j < SPT; ++j) {
          // warp-exclusive scan of m[j]; the common case (every m <= 1) is one ballot
          uint32_t excl, wtot;
          if (__all_sync(0xffffffffu, m[j] <= 1)) {
            const uint32_t b = __ballot_sync(0xffffffffu, m[j] != 0);
            excl = __popc(b & lanemask_lt());
            wtot = __popc(b);
          } else {
            uint32_t x = m[j];
            #pragma unroll
            for (int o = 1; o < 32; o <<= 1) {
              const uint32_t y = __shfl_up_sync(0xffffffffu, x, o);
              if (lane >= o) x += y;
            }
            excl = x - m[j];
            wtot = __shfl_sync(0xffffffffu, x, 31);
          }
          if (wtot == 0) continue;
          uint32_t wb = 0;
          if (lane == 0) wb = atomicAdd(&s_wcur, wtot);
          wb = __shfl_sync(0xffffffffu, wb, 0);
          unsigned long long pos = gbase + wb + excl;
          if (m[j] == 1) {
            if (pos < P.out_cap) {
              out_r[pos] = rfirst[j];
              out_s[pos] = sp[j];
            }
          } else if (m[j] > 1) {
            for (uint32_t i = s_head[slot_of(sk[j], H)]; i != NIL16; i = s_next[i]) {
              const T r = s_rt[i];
              if (TT::key(r) == sk[j]) {
                if (pos < P.out_cap) {
                  out_r[pos] = TT::pay(r);
                  out_s[pos] = sp[j];
                }
                ++pos;
              }
            }
          }
        }
        bar_compute(NT);  // s_base / s_wcur are reused by the next round
      }
    }
    __syncthreads();  // end of item: s_rt / s_head are rewritten, s_jobs[it+1] is ready
  }

  // ---- aggregate: warp shuffle reduce, then one 64-bit atomic per block --------
  #pragma unroll
  for (int o = 16; o; o >>= 1) {
    my_cnt += __shfl_xor_sync(0xffffffffu, my_cnt, o);
    my_chk += __shfl_xor_sync(0xffffffffu, my_chk, o);
  }
  if (lane == 0) {
    s_red[0][warp] = my_cnt;
    s_red[1][warp] = my_chk;
  }
  __syncthreads();
  if (threadIdx.x == 0) {
    unsigned long long c = 0, h = 0;
    for (int w = 0; w < NT / 32 + 1; ++w) {
      c += s_red[0][w];
      h += s_red[1][w];
    }
    if (c) {
      atomicAdd(&P.results[RES_MATCHES], c);
      atomicAdd(&P.results[RES_CHECKSUM], h);
    }
  }
}

}  // namespace hj
