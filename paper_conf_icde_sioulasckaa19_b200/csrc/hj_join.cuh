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

#include <type_traits>

namespace hj {


struct JoinJob {
  uint32_t item, nr, shift;  // shift: tuples between the 16-byte aligned copy start and rb
  unsigned long long rb, sb, se;
};


// Claim the next work item and decode it (item -> co-partition q by binary search over the
// planner's item prefix; then the R chunk and S chunk of q it covers). One lane.
// SWAP: an item of a swapped co-partition (P.ist2): the build chunk is its S side (one chunk), the
// probe chunk one C_S-sized chunk of its R side.
template <typename T, bool SWAP = false>
__device__ __forceinline__ JoinJob claim_job(const Plan& P, uint32_t total_items) {
  JoinJob j;
  j.item = atomicAdd(&P.counters[SWAP ? CNT_NEXT_ITEM2 : CNT_NEXT_ITEM], 1u);
  j.nr = j.shift = 0;
  j.rb = j.sb = j.se = 0;
  if (j.item < total_items) {
    const uint32_t np = 1u << P.B;
    const uint32_t* ist = SWAP ? P.ist2 : P.ist;
    uint32_t lo = 0, hi = np;  // largest q with ist[q] <= item
    while (hi - lo > 1) {
      const uint32_t mid = (lo + hi) >> 1;
      if (ist[mid] <= j.item) lo = mid; else hi = mid;
    }
    const uint32_t q = lo;
    if (!SWAP && P.bc) {  // bucket chains (NEXT-1): item = (R slice, S slice) of q, slices from k_bc_slices
      const uint32_t loc = j.item - P.ist[q], nsch = P.bc_rel[1].sst[q + 1] - P.bc_rel[1].sst[q];
      const uint4 rs = P.bc_rel[0].sl[P.bc_rel[0].sst[q] + loc / nsch];
      const uint4 ss = P.bc_rel[1].sl[P.bc_rel[1].sst[q] + loc % nsch];
      j.rb = ((unsigned long long)rs.y << 32) | rs.x;
      j.nr = rs.z;
      j.sb = ((unsigned long long)ss.y << 32) | ss.x;
      j.se = j.sb + ss.z;
      const uintptr_t a = reinterpret_cast<uintptr_t>((const T*)P.rel[0].t2 + j.rb);
      j.shift = (uint32_t)((a & 15) / sizeof(T));
      return j;
    }
    // build side (rel SWAP) and probe side (rel !SWAP)
    const unsigned long long r0 = P.rel[SWAP ? 1 : 0].off[q], rn = P.rel[SWAP ? 1 : 0].off[q + 1] - r0;
    const unsigned long long s0 = P.rel[SWAP ? 0 : 1].off[q], sn = P.rel[SWAP ? 0 : 1].off[q + 1] - s0;
    // probe chunks: C_S tuples; swapped items probe R chunks of 2^lgCRp <= C_R tuples (more items:
    // a duplicate-heavy probe side keeps many blocks busy)
    const unsigned long long CSx = SWAP ? 1ull << P.lgCRp : (unsigned long long)P.CS;
    const unsigned long long nsch = (sn + CSx - 1) / CSx;
    const unsigned long long loc = j.item - ist[q];
    const unsigned long long rc = loc / nsch, sc = loc % nsch;
    j.rb = r0 + rc * P.CR;
    j.nr = (uint32_t)min((unsigned long long)P.CR, rn - rc * P.CR);
    j.sb = s0 + sc * CSx;
    j.se = j.sb + min(CSx, sn - sc * CSx);
    const uintptr_t a = reinterpret_cast<uintptr_t>((const T*)P.rel[SWAP ? 1 : 0].t2 + j.rb);
    j.shift = (uint32_t)((a & 15) / sizeof(T));  // tuples between the 16 B aligned copy start and rb
  }
  return j;
}

// TMA bulk copy of a job's R chunk (the 16-byte aligned superset) into an smem tile buffer.
template <typename T, bool SWAP = false>
__device__ __forceinline__ void issue_r_copy(const Plan& P, const JoinJob& j, T* buf, unsigned long long* bar) {
  const uintptr_t a = reinterpret_cast<uintptr_t>((const T*)P.rel[SWAP ? 1 : 0].t2 + j.rb);
  const uintptr_t a0 = a & ~(uintptr_t)15;
  const uint32_t bytes = (uint32_t)(((a + (uintptr_t)j.nr * sizeof(T) - a0) + 15) & ~(uintptr_t)15);
  fence_proxy_async();  // prior generic-proxy reads of buf (the item before last) are ordered before
  mbar_arrive_expect_tx(bar, bytes);
  bulk_g2s(buf, reinterpret_cast<const void*>(a0), bytes, bar);
}

// L2 prefetch of a claimed item's R chunk and first probe round (TMA prefetch, no smem): the
// R copy issued after the end-of-item barrier and the first S loads then hit L2.
template <typename T, bool SWAP = false>
__device__ __forceinline__ void prefetch_item_l2(const Plan& P, const JoinJob& j, uint32_t s_round) {
  auto pf = [](const T* b, unsigned long long n) {
    const uintptr_t a = reinterpret_cast<uintptr_t>(b), a0 = a & ~(uintptr_t)15;
    const uintptr_t a1 = (a + n * sizeof(T) + 15) & ~(uintptr_t)15;
    if (a1 > a0) bulk_prefetch_l2(reinterpret_cast<const void*>(a0), (uint32_t)(a1 - a0));
  };
  pf((const T*)P.rel[SWAP ? 1 : 0].t2 + j.rb, j.nr);
  pf((const T*)P.rel[SWAP ? 0 : 1].t2 + j.sb, min((unsigned long long)s_round, j.se - j.sb));
}

// a tuple of the R tile from its 32-bit shared-window address (keeps the tile base in a register:
// through the generic pointer the compiler rematerialized the shared-window base per access)
__device__ __forceinline__ unsigned long long lds_tuple(uint32_t a, unsigned long long*) {
  unsigned long long v;
  asm volatile("ld.shared.u64 %0, [%1];" : "=l"(v) : "r"(a));
  return v;
}
__device__ __forceinline__ ulonglong2 lds_tuple(uint32_t a, ulonglong2*) {
  ulonglong2 v;
  asm volatile("ld.shared.v2.u64 {%0, %1}, [%2];" : "=l"(v.x), "=l"(v.y) : "r"(a));
  return v;
}

__device__ __forceinline__ uint32_t lds_u32(uint32_t a) {
  uint32_t v;
  asm volatile("ld.shared.u32 %0, [%1];" : "=r"(v) : "r"(a));
  return v;
}
__device__ __forceinline__ uint32_t lds_u16(uint32_t a) {
  unsigned short v;
  asm volatile("ld.shared.u16 %0, [%1];" : "=h"(v) : "r"(a));
  return v;
}

__device__ __forceinline__ void bar_compute(int nthreads) {  // named barrier 1: compute warps only
  asm volatile("barrier.sync 1, %0;" ::"r"(nthreads) : "memory");
}
// end-of-item barrier of the whole block (compute warps + scheduler warp), reached from two code
// sites: the non-aligned barrier.sync with an explicit thread count is defined for divergent
// arrival (bar.sync / __syncthreads are .aligned)
__device__ __forceinline__ void bar_item(int nthreads) { asm volatile("barrier.sync 2, %0;" ::"r"(nthreads) : "memory"); }

// Block = NT compute threads + one scheduler warp. The scheduler warp claims and decodes item
// k+1 and starts its R chunk's TMA bulk copy into the other half of a double-buffered smem tile
// while the compute warps join item k; it only joins the end-of-item barrier. So neither the
// dependent global loads of the item lookup nor the R-chunk load sit on the join's critical path.
//
// Output of the materialized mode: per probe round every thread knows the match count of each
// of its S tuples (first chain walk, which also keeps the first match's payload); each warp
// reserves its round's pairs with ONE global atomicAdd (no block barrier in the round: c3 join
// 0.690 -> 0.675 ms against one atomic per block and round behind two barriers), and its lanes
// write their pairs at warp-contiguous positions (coalesced stores). This replaces the paper's
// per-warp buffer + global atomic per flush. Chains are re-walked only for S tuples
// with more than one match.
// RBUF = 2: the next item's R chunk is copied while the current item is joined (double buffer);
// RBUF = 1: it is copied right after the end-of-item barrier (less smem -> more blocks per SM).
// 16-bit wait-free push-front for H16 heads: a 16-bit CAS loop (retries only when two R tuples
// of the same slot insert at the same time)
__device__ __forceinline__ uint32_t exch16(unsigned short* a, uint32_t v) {
  unsigned short old = *a, assumed;
  do {
    assumed = old;
    old = atomicCAS(a, assumed, (unsigned short)v);
  } while (old != assumed);
  return old;
}

// H16: 16-bit chain heads (half the head array -> one more block per SM fits in shared memory)
// PF: the next probe round's S tuples are loaded (into registers) before the current round's
// chains are walked, so the S load latency overlaps the walk instead of opening each round.
// SPF > 0: the S chunk is streamed through L2 ahead of the probe: at the item's first round one
// compute thread issues a TMA L2 prefetch of rounds 1..SPF, then at round k of rounds k+SPF (one
// cp.async.bulk.prefetch.L2 of NT*SPT tuples per round), so the bytes in flight per SM no longer
// depend on the registers of the probing threads.
// F2: the cheaper slot hash (slot_of2; the host picks it for 8-byte keys and for 4-byte keys whose
// bits above B fit in 2 lg bits). BF: branch-free first chain step for all SPT tuples of a round.
// the pair signature of (build tuple, probe tuple) payloads: sig(r_pay, s_pay) (SWAP: the build
// side is S)
template <bool SWAP>
__device__ __forceinline__ uint64_t sig_bp(uint64_t build_pay, uint64_t probe_pay) {
  return SWAP ? pair_sig(probe_pay, build_pay) : pair_sig(build_pay, probe_pay);
}

template <typename K, int NT, int SPT, bool MAT, int RBUF, bool H16 = false, bool PF = false, bool L2PF = false,
          int SPF = 0, bool F2 = false, bool BF = true, bool SWAP = false>
__device__ __forceinline__ void join_body(const Plan& P) {
  using TT = Tup<K>;
  using T = typename TT::T;
  extern __shared__ __align__(16) unsigned char s_raw[];
  const SlotHash H = P.H;
  const uint32_t nb = 1u << H.lg;
  const uint32_t cap = (P.CR + 3) & ~1u;  // tile buffer in tuples: +2 for the aligned superset, even -> 16 B aligned
  T* s_rtb = reinterpret_cast<T*>(s_raw);                             // RBUF x cap tuples
  using HT = typename std::conditional<H16, unsigned short, uint32_t>::type;
  HT* s_head = reinterpret_cast<HT*>(s_rtb + RBUF * cap);             // nb
  uint16_t* s_next = reinterpret_cast<uint16_t*>(s_head + nb);       // CR + 1
  // chain end. SENT (count mode with the branch-free first step): the sentinel index CR, so an
  // empty slot's "tuple" s_rt[CR] is the tile's spare slot (read and discarded) and s_next[CR] = CR:
  // the probe step needs no selects (c2 join 0.628 -> 0.589 ms). Materialize mode keeps 0xffff and
  // the selects (the sentinel cost it a spill at 72 registers: c3 0.690 -> 0.707)
  constexpr bool SENT = BF && !MAT;
  const uint32_t NIL = SENT ? P.CR : 0xffffu;
  // SENT: shared addresses as base + index * size with the sizes runtime values (P.one == 1), so
  // they are IMADs on the FMA pipe rather than LEAs on the ALU pipe (the count probe is ALU-bound)
  const uint32_t tmul = (uint32_t)sizeof(T) * P.one, hmul = (uint32_t)sizeof(HT) * P.one, nmul = 2u * P.one;
  const uint32_t s_head_sh = (uint32_t)__cvta_generic_to_shared(s_head);
  const uint32_t s_next_sh = (uint32_t)__cvta_generic_to_shared(s_next);
  __shared__ JoinJob s_jobs[2];
  __shared__ __align__(8) unsigned long long s_bar[2];
  __shared__ unsigned long long s_red[2][NT / 32 + 1];

  const uint32_t total_items = (SWAP ? P.ist2 : P.ist)[1u << P.B];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const bool sched = threadIdx.x >= NT;
  K* out_r = (K*)P.out_r;
  K* out_s = (K*)P.out_s;
  const T* ssrc = (const T*)P.rel[SWAP ? 0 : 1].t2;  // the probe side
  unsigned long long my_cnt = 0, my_chk = 0;
  uint32_t my_cnt32 = 0;  // count mode: this thread's matches in the current round
  // checksum in MATERIALIZE mode too (block-uniform; the pairs' signatures are summed in the first
  // chain walk, so re-walks of multi-match tuples only write)
  const bool chk = !MAT || P.mat_chk != 0;

  if (threadIdx.x == NT) {
    mbar_init(&s_bar[0], 1);
    mbar_init(&s_bar[1], 1);
    fence_mbar_init();
    JoinJob j = claim_job<T, SWAP>(P, total_items);
    if (j.item < total_items) issue_r_copy<T, SWAP>(P, j, s_rtb, &s_bar[0]);
    s_jobs[0] = j;
  }
  __syncthreads();

  for (uint32_t it = 0;; ++it) {
    const JoinJob job = s_jobs[it & 1];
    if (job.item >= total_items) break;
    if (sched) {
      JoinJob j;
      if (lane == 0) {
        j = claim_job<T, SWAP>(P, total_items);
        if (L2PF && RBUF == 1 && j.item < total_items) prefetch_item_l2<T, SWAP>(P, j, NT * SPT);
        if (RBUF == 2 && j.item < total_items)
          issue_r_copy<T, SWAP>(P, j, s_rtb + ((it + 1) & 1) * cap, &s_bar[(it + 1) & 1]);
        s_jobs[(it + 1) & 1] = j;
      }
      bar_item(NT + 32);  // end-of-item barrier (matches the compute warps' one below)
      if (RBUF == 1 && lane == 0 && j.item < total_items) issue_r_copy<T, SWAP>(P, j, s_rtb, &s_bar[(it + 1) & 1]);
      continue;
    }

    // ---- first probe round's S loads (in flight during the build) --------------------------
    // S offsets are 32-bit, relative to the item's first S tuple (an item has <= C_S < 2^31)
    constexpr uint32_t RND = (uint32_t)NT * SPT;
    const T* const sitem = ssrc + job.sb + threadIdx.x;
    const uint32_t slen = (uint32_t)(job.se - job.sb);
    K sk[SPT], sp[SPT];
    auto load_s = [&](uint32_t off) {
      const uint32_t rem = min(slen - off, RND);
      #pragma unroll
      for (int j = 0; j < SPT; ++j) {
        if ((uint32_t)(j * NT) + threadIdx.x < rem) {
          const T t = __ldcs(sitem + off + j * NT);
          sk[j] = TT::key(t);
          sp[j] = TT::pay(t);
        }
      }
    };
    T nx[PF ? SPT : 1];  // PF: the next round's tuples
    auto load_next = [&](uint32_t off) {
      const uint32_t rem = min(slen - off, RND);
      #pragma unroll
      for (int j = 0; j < SPT; ++j)
        if ((uint32_t)(j * NT) + threadIdx.x < rem) nx[j] = __ldcs(sitem + off + j * NT);
    };
    load_s(0);
    for (uint32_t i = threadIdx.x; i < nb; i += NT) s_head[i] = (HT)NIL;
    if (SENT && threadIdx.x == 0) s_next[NIL] = (uint16_t)NIL;
    const T* s_rt = s_rtb + (RBUF == 2 ? (it & 1) * cap : 0) + job.shift;
    const uint32_t s_rt_sh = (uint32_t)__cvta_generic_to_shared(s_rt);
    mbar_wait(&s_bar[it & 1], (it >> 1) & 1);  // R chunk landed (TMA)
    bar_compute(NT);
    // ---- build (a6): wait-free push-front insert (Listing 2) ----------------------
    for (uint32_t i = threadIdx.x; i < job.nr; i += NT) {
      const K k = TT::key(lds_tuple(s_rt_sh + i * (uint32_t)sizeof(T), (T*)nullptr));
      s_next[i] = H16 ? (uint16_t)exch16(reinterpret_cast<unsigned short*>(&s_head[slot_for<F2>(k, H)]), i)
                      : (uint16_t)atomicExch(reinterpret_cast<uint32_t*>(&s_head[slot_for<F2>(k, H)]), i);
    }
    bar_compute(NT);

    // ---- probe (a7) + output (a8), SPT tuples per thread per round --------------------------
    for (uint32_t off = 0; off < slen; off += RND) {
      if (SPF > 0 && threadIdx.x == 0) {
        const uint32_t lo = off == 0 ? RND : off + SPF * RND;
        const uint32_t hi = min(off + (SPF + 1) * RND, slen);
        if (lo < hi) {
          const T* sbase = ssrc + job.sb;
          const uintptr_t a = reinterpret_cast<uintptr_t>(sbase + lo), a0 = a & ~(uintptr_t)15;
          const uintptr_t a1 = (reinterpret_cast<uintptr_t>(sbase + hi) + 15) & ~(uintptr_t)15;
          bulk_prefetch_l2(reinterpret_cast<const void*>(a0), (uint32_t)(a1 - a0));
        }
      }
      if (PF) {
        if (off != 0) {
          #pragma unroll
          for (int j = 0; j < SPT; ++j) {
            sk[j] = TT::key(nx[j]);
            sp[j] = TT::pay(nx[j]);
          }
        }
        if (off + RND < slen) load_next(off + RND);
      } else if (off != 0) {
        load_s(off);
      }
      uint32_t idx[SPT], m[SPT];
      K rfirst[SPT];
      // this round's tuples; a full round needs no per-tuple bounds (block-uniform branch)
      const uint32_t rem = min(slen - off, RND);
      if (rem == RND) {
        #pragma unroll
        for (int j = 0; j < SPT; ++j)
          idx[j] = SENT ? (H16 ? lds_u16(s_head_sh + slot_for<F2>(sk[j], H) * hmul) : lds_u32(s_head_sh + slot_for<F2>(sk[j], H) * hmul))
                        : (uint32_t)s_head[slot_for<F2>(sk[j], H)];
      } else {
        #pragma unroll
        for (int j = 0; j < SPT; ++j)
          idx[j] = ((uint32_t)(j * NT) + threadIdx.x < rem) ? (uint32_t)s_head[slot_for<F2>(sk[j], H)] : NIL;
      }
      #pragma unroll
      for (int j = 0; j < SPT; ++j) m[j] = 0;
      // first chain step of every tuple without branches (unique build keys: chains of length
      // <= 1, so this is usually the whole probe): the head's tuple is read even for an empty
      // slot (index 0 instead, discarded), the signature is computed for every tuple and added
      // only on a hit; the general walk below runs only while some lane still has a chain.
      // BF = false (the round-1 8-byte shape, one tuple per thread): every step branchy.
      bool live = !BF;
      #pragma unroll
      for (int j = 0; j < SPT && BF; ++j) {
        const bool v = idx[j] != NIL;
        const uint32_t i0 = SENT ? idx[j] : (v ? idx[j] : 0u);  // SENT: NIL reads the spare slot (discarded)
        const T r = lds_tuple(s_rt_sh + i0 * (SENT ? tmul : (uint32_t)sizeof(T)), (T*)nullptr);
        const bool hit = v && TT::key(r) == sk[j];
        if (MAT) rfirst[j] = TT::pay(r);
        if (!MAT || chk) {
          const uint64_t sg = sig_bp<SWAP>((uint64_t)TT::pay(r), (uint64_t)sp[j]);
          if (hit) my_chk += sg;  // predicated add (no selects)
        }
        if (MAT) m[j] = hit ? 1u : 0u;
        else if (hit) ++my_cnt32;  // count mode: one predicated add, no per-tuple match counts
        idx[j] = SENT ? lds_u16(s_next_sh + i0 * nmul) : (v ? (uint32_t)s_next[i0] : NIL);  // SENT: s_next[NIL] = NIL
        live |= idx[j] != NIL;
      }
      // chains of all SPT tuples advance together (independent shared-memory loads in flight)
      if constexpr (BF) {
        while (__any_sync(0xffffffffu, live)) {
          live = false;
          #pragma unroll
          for (int j = 0; j < SPT; ++j) {
            if (idx[j] != NIL) {
              const T r = lds_tuple(s_rt_sh + idx[j] * (uint32_t)sizeof(T), (T*)nullptr);
              if (TT::key(r) == sk[j]) {
                if (MAT && m[j] == 0) rfirst[j] = TT::pay(r);
                if (!MAT || chk) my_chk += sig_bp<SWAP>((uint64_t)TT::pay(r), (uint64_t)sp[j]);
                if (MAT) ++m[j];
                else ++my_cnt32;
              }
              idx[j] = s_next[idx[j]];
              live |= idx[j] != NIL;
            }
          }
        }
      } else {
        // branchy walk (BF = false): the lanes of a warp walk chains of different lengths, so the
        // walk body runs max-chain times per warp; it only keeps the first match's payload (later
        // matches of duplicate R keys add their signatures at once, rarely), and the signature of
        // the first match is computed once after the walk, by all lanes together
        while (live) {
          live = false;
          #pragma unroll
          for (int j = 0; j < SPT; ++j) {
            if (idx[j] != NIL) {
              const T r = lds_tuple(s_rt_sh + idx[j] * (uint32_t)sizeof(T), (T*)nullptr);
              if (TT::key(r) == sk[j]) {
                if (m[j] == 0) rfirst[j] = TT::pay(r);
                else if (!MAT || chk) my_chk += sig_bp<SWAP>((uint64_t)TT::pay(r), (uint64_t)sp[j]);
                ++m[j];
              }
              idx[j] = s_next[idx[j]];
              live |= idx[j] != NIL;
            }
          }
        }
        #pragma unroll
        for (int j = 0; j < SPT; ++j) {
          if (!MAT || chk) {
            const uint64_t sg = sig_bp<SWAP>((uint64_t)rfirst[j], (uint64_t)sp[j]);
            if (m[j]) my_chk += sg;
          }
          if (!MAT) my_cnt32 += m[j];
        }
      }
      if (!MAT) {  // a round adds < SPT * C_R <= 2^20 matches per thread
        my_cnt += my_cnt32;
        my_cnt32 = 0;
      }
      if (MAT) {
        uint32_t mt = 0;
        #pragma unroll
        for (int j = 0; j < SPT; ++j) mt += m[j];
        my_cnt += mt;
        const uint32_t wsum = __reduce_add_sync(0xffffffffu, mt);
        unsigned long long wb = 0;  // this warp's output range for the round: one global atomic
        if (lane == 0 && wsum) wb = atomicAdd(&P.results[RES_CURSOR], (unsigned long long)wsum);
        const unsigned long long rbase = __shfl_sync(0xffffffffu, wb, 0);
        K* const o_r = out_r + rbase;
        K* const o_s = out_s + rbase;
        const uint32_t room = rbase >= P.out_cap ? 0u : (uint32_t)min(P.out_cap - rbase, 0xffffffffull);
        // positions relative to the warp's base: 32-bit (a round emits < 2^32 pairs)
        uint32_t pos0 = 0;
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
          uint32_t pos = pos0 + excl;
          pos0 += wtot;
          if (m[j] == 1) {
            if (pos < room) {
              o_r[pos] = SWAP ? sp[j] : rfirst[j];
              o_s[pos] = SWAP ? rfirst[j] : sp[j];
            }
          } else if (m[j] > 1) {
            for (uint32_t i = s_head[slot_for<F2>(sk[j], H)]; i != NIL; i = s_next[i]) {
              const T r = s_rt[i];
              if (TT::key(r) == sk[j]) {
                if (pos < room) {
                  o_r[pos] = SWAP ? sp[j] : TT::pay(r);
                  o_s[pos] = SWAP ? TT::pay(r) : sp[j];
                }
                ++pos;
              }
            }
          }
        }
      }
    }
    bar_item(NT + 32);  // end of item: the tile buffer and s_head are reused, s_jobs[it+1] is ready
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

template <typename K, int NT, int SPT, bool MAT, int MINB, int RBUF, bool H16 = false, bool PF = false,
          bool L2PF = false, int SPF = 0, bool F2 = false, bool BF = true>
__global__ void __launch_bounds__(NT + 32, MINB) k_join(Plan P) {
  pdl_wait();
  join_body<K, NT, SPT, MAT, RBUF, H16, PF, L2PF, SPF, F2, BF>(P);
  if (P.ist2 != nullptr && !P.bc) {  // then the swapped items (usually none: one load, then exit)
    __syncthreads();
    join_body<K, NT, SPT, MAT, RBUF, H16, PF, L2PF, SPF, F2, BF, true>(P);
  }
}

}  // namespace hj
