// hj_partition.cuh -- steps a1-a4 of the hot path:
//   k_hist   a1: histogram of p = key & (2^B-1) for both relations (shared-memory counters)
//   k_plan   a2/a5: one-block scan -> co-partition offsets, pass cursors, pass-2 chunk list,
//            join work list
//   k_pass   a3 (MODE 1, SoA tiles -> T1 by d1) and a4 (MODE 2, chunks of each pass-1
//            partition -> T2 by d2)
//
// Partitioning follows PAPER.md §III-A: a multi-pass radix partition whose
// fan-out per pass is bounded by the shared memory holding per-partition metadata and the
// shuffle space used to make the device-memory writes coalesced. Each pass
// stages a whole tile in shared memory sorted by digit, then writes every digit's run to a
// range reserved with one global atomic per (tile, digit) -- the histogram-derived cursors
// replace the paper's bucket chains (reading D2 in DESIGN.md).
#pragma once
#include "hj_common.cuh"
#include "hj_plan.cuh"

namespace hj {

// ------------------------------------------------------------------------------------------
// a1: histogram. grid = (blocks_per_rel, 2). Each block counts a contiguous, 16-byte aligned
// range of one relation's keys in 2^B shared-memory counters (smem atomics measured at ~6
// tuples/clk/SM on B200, tools/microbench/mb_rank.cu), then merges non-zero counters with
// one global RED each. For B > 15 (more than 128 KB of counters) SMEM = false counts with
// global atomics directly (correct, slower; not used by the benchmark configs).
// ------------------------------------------------------------------------------------------
template <typename K, bool SMEM>
__global__ void __launch_bounds__(1024) k_hist(Plan P) {
  extern __shared__ uint32_t s_hist[];
  const int rel = blockIdx.y;
  const RelDev& R = P.rel[rel];
  const unsigned long long n = R.n;
  const uint32_t np = 1u << P.B;
  const uint32_t mask = np - 1;
  if (SMEM) {
    for (uint32_t i = threadIdx.x; i < np; i += blockDim.x) s_hist[i] = 0;
    __syncthreads();
  }
  uint32_t* h = SMEM ? s_hist : R.cnt;
  // counters are indexed by q = (p & (2^b1-1)) << b2 | p >> b1, the planner's order
  const int b1 = P.b1, b2 = P.b2;
  const uint32_t mb1 = (1u << b1) - 1;
  auto bin = [&](uint32_t p) -> uint32_t { return ((p & mb1) << b2) | (p >> b1); };
  constexpr int VEC = 16 / sizeof(K);
  unsigned long long per = (n + gridDim.x - 1) / gridDim.x;
  per = (per + VEC - 1) / VEC * VEC;
  const unsigned long long lo = (unsigned long long)blockIdx.x * per;
  const unsigned long long hi = lo + per < n ? lo + per : n;
  const K* keys = (const K*)R.keys;
  if (lo < hi) {
    const bool aligned = ((reinterpret_cast<uintptr_t>(keys) & 15) == 0);
    unsigned long long i = lo;
    if (aligned) {
      const unsigned long long nvec = (hi - lo) / VEC;
      const uint4* kv = reinterpret_cast<const uint4*>(keys + lo);
      constexpr int U = 4;  // 4 x 16 B loads in flight per thread before the atomics
      unsigned long long v = threadIdx.x;
      for (; v + (U - 1) * blockDim.x < nvec; v += U * blockDim.x) {
        uint4 x[U];
        #pragma unroll
        for (int u = 0; u < U; ++u) x[u] = __ldcs(kv + v + u * blockDim.x);
        #pragma unroll
        for (int u = 0; u < U; ++u) {
          const K* e = reinterpret_cast<const K*>(&x[u]);
          #pragma unroll
          for (int t = 0; t < VEC; ++t) atomicAdd(&h[bin((uint32_t)(e[t]) & mask)], 1u);
        }
      }
      for (; v < nvec; v += blockDim.x) {
        uint4 x = __ldcs(kv + v);
        const K* e = reinterpret_cast<const K*>(&x);
        #pragma unroll
        for (int t = 0; t < VEC; ++t) atomicAdd(&h[bin((uint32_t)(e[t]) & mask)], 1u);
      }
      i = lo + nvec * VEC;
    }
    for (unsigned long long j = i + threadIdx.x; j < hi; j += blockDim.x) atomicAdd(&h[bin((uint32_t)keys[j] & mask)], 1u);
  }
  if (SMEM) {
    __syncthreads();
    for (uint32_t i = threadIdx.x; i < np; i += blockDim.x) {
      uint32_t c = s_hist[i];
      if (c) atomicAdd(&R.cnt[i], c);
    }
  }
}

// ------------------------------------------------------------------------------------------
// a2 + a5: the planner. One block of 1024 threads; 2^B <= 2^20 entries per relation.
//   off[q]  = exclusive scan of cnt[p(q)] in q-order          (co-partition starts, T2)
//   cur1[d1] = off[d1 << b2], cur2[q] = off[q]                (pass reservation cursors)
//   cst[d1]  = exclusive scan of ceil(|partition d1| / C2)    (pass-2 chunk list)
//   ist[q]   = exclusive scan of items(q),  items(q) = ceil(|R_q|/CR) * ceil(|S_q|/CS) if both
//              non-empty else 0                                (join work list)
// ------------------------------------------------------------------------------------------
__device__ __forceinline__ uint32_t q_to_p(uint32_t q, int b1, int b2) {
  const uint32_t d1 = q >> b2, d2 = q & ((1u << b2) - 1);
  return (d2 << b1) | d1;
}

__device__ __forceinline__ unsigned long long plan_items(const Plan& P, uint32_t cr, uint32_t cs) {
  return (cr && cs) ? (unsigned long long)((cr + P.CR - 1) / P.CR) * ((cs + P.CS - 1) / P.CS) : 0ull;
}

// grid = ceil(2^B / 1024) blocks; block b owns q in [1024 b, 1024 (b+1)), one q per thread, so
// every store is coalesced. Each block first sums all counts below its range itself (a redundant
// prefix: at most 2^B / 1024 independent loads per thread, L2-resident), then scans its own
// range. The last block to finish (atomic ticket) builds the pass-2 chunk lists.
__global__ void __launch_bounds__(1024) k_plan(Plan P) {
  constexpr int NT = 1024;
  __shared__ unsigned long long s_tmp[NT / 32 + 1];
  __shared__ bool s_last;
  const uint32_t np = 1u << P.B;
  const uint32_t F1 = 1u << P.b1;
  const uint32_t b = blockIdx.x;
  // ---- prefix of everything below this block's range -------------------------------------
  unsigned long long sR = 0, sS = 0, sI = 0;
  #pragma unroll 8
  for (uint32_t k = 0; k < b; ++k) {
    const uint32_t cr = P.rel[0].cnt[k * NT + threadIdx.x], cs = P.rel[1].cnt[k * NT + threadIdx.x];
    sR += cr;
    sS += cs;
    sI += plan_items(P, cr, cs);
  }
  unsigned long long tot;
  block_exclusive_scan64<NT>(sR, s_tmp, &tot);
  unsigned long long bR = tot;
  block_exclusive_scan64<NT>(sS, s_tmp, &tot);
  unsigned long long bS = tot;
  block_exclusive_scan64<NT>(sI, s_tmp, &tot);
  unsigned long long bI = tot;
  // ---- own range ---------------------------------------------------------------------------
  const uint32_t q = b * NT + threadIdx.x;
  uint32_t cr = 0, cs = 0;
  if (q < np) {
    cr = P.rel[0].cnt[q];
    cs = P.rel[1].cnt[q];
  }
  unsigned long long tR, tS, tI;
  const unsigned long long oR = bR + block_exclusive_scan64<NT>(cr, s_tmp, &tR);
  const unsigned long long oS = bS + block_exclusive_scan64<NT>(cs, s_tmp, &tS);
  const unsigned long long oI = bI + block_exclusive_scan64<NT>(plan_items(P, cr, cs), s_tmp, &tI);
  if (q < np) {
    P.rel[0].off[q] = oR;
    P.rel[0].cur2[q] = oR;
    P.rel[1].off[q] = oS;
    P.rel[1].cur2[q] = oS;
    P.ist[q] = (uint32_t)oI;
  }
  if (b == gridDim.x - 1 && threadIdx.x == 0) {
    P.rel[0].off[np] = bR + tR;
    P.rel[1].off[np] = bS + tS;
    P.ist[np] = (uint32_t)(bI + tI);
  }
  // ---- last block: pass-2 chunk lists over the 2^b1 pass-1 partitions (b1 <= 10) ----------
  __threadfence();
  __syncthreads();
  if (threadIdx.x == 0) s_last = atomicAdd(&P.counters[CNT_PLAN_DONE], 1u) == gridDim.x - 1;
  __syncthreads();
  if (!s_last) return;
  __threadfence();
  for (int rel = 0; rel < 2; ++rel) {
    const RelDev& R = P.rel[rel];
    unsigned long long nch = 0;
    if (threadIdx.x < F1) {
      const unsigned long long a = __ldcg(&R.off[(unsigned long long)threadIdx.x << P.b2]);
      const unsigned long long e = __ldcg(&R.off[(unsigned long long)(threadIdx.x + 1) << P.b2]);
      R.cur1[threadIdx.x] = a;
      nch = (e - a + P.C2 - 1) / P.C2;
    }
    const unsigned long long cb = block_exclusive_scan64<NT>(nch, s_tmp, &tot);
    if (threadIdx.x < F1) R.cst[threadIdx.x] = (uint32_t)cb;
    if (threadIdx.x == 0) R.cst[F1] = (uint32_t)tot;
  }
}

// ------------------------------------------------------------------------------------------
// a3 / a4: one partition pass. One persistent block of NT = 1024 threads per SM loops over
// work units:
//   MODE 1: unit = a tile of TILE consecutive rows of the SoA input of R or S; digit
//           d1 = key & (2^b1 - 1); output T1 at cur1[d1] reservations.
//   MODE 2: unit = chunk k of pass-1 partition d1 (T1[off + k*TILE, ...)); digit
//           d2 = (key >> b1) & (2^b2 - 1); output T2 at cur2[d1 << b2 | d2] reservations.
// Per unit: rank every tuple within its digit with a shared-memory atomicAdd (returning the
// rank; measured ~6 tuples/clk/SM), scan the per-digit counts, reserve each digit's run in the
// output with one global atomicAdd, shuffle the tile into digit order in shared memory, then
// stream it out so consecutive threads write consecutive addresses of a run (P:142-148
// coalescing, P:269-272 shuffle space); L2 merges the partial lines at run boundaries, so
// DRAM sees full lines (ncu: DRAM bytes == algorithmic bytes).
// Latency hiding: the NEXT unit's loads are issued into registers before the current unit is
// ranked (they stay in flight across its barriers), and each reservation atomic's result is
// consumed only after the shared-memory shuffle.
// Every output slot is written exactly once; order inside a run is whatever the shared-memory
// atomics produced (partitions are multisets, reading S9).
// ------------------------------------------------------------------------------------------
template <typename K>
struct PassUnit {
  const void* src_k;  // MODE 1: key column at the unit start; MODE 2: first AoS tuple of the unit
  const void* src_p;  // MODE 1: payload column at the unit start
  void* dst;          // output buffer (T1 or T2) of the unit's relation
  unsigned long long* cur;  // reservation cursors: cur1 (MODE 1) or &cur2[d1 << b2] (MODE 2)
  uint32_t len;
};

// Round-robin unit walker: unit u = blockIdx.x + k * gridDim.x. MODE 2 keeps the current
// (relation, d1) and advances d1 through the shared-memory chunk prefix instead of searching.
template <typename K, int MODE, int TILE>
struct UnitWalker {
  unsigned long long units0, units;
  int rel;
  uint32_t d1;
  __device__ __forceinline__ bool get(const Plan& P, unsigned long long u, PassUnit<K>& U, const uint32_t* s_cst,
                                      const unsigned long long* s_pst) {
    using T = typename Tup<K>::T;
    if (u >= units) return false;
    const int r = (u < units0) ? 0 : 1;
    const unsigned long long ul = r ? u - units0 : u;
    const RelDev& R = P.rel[r];
    if (MODE == 1) {
      const unsigned long long s0 = ul * TILE;
      U.src_k = (const K*)R.keys + s0;
      U.src_p = (const K*)R.pays + s0;
      U.dst = R.t1;
      U.cur = R.cur1;
      U.len = (uint32_t)min((unsigned long long)TILE, R.n - s0);
    } else {
      if (r != rel) {
        rel = r;
        d1 = 0;
      }
      const uint32_t* cst = s_cst + r * 1025;
      while (cst[d1 + 1] <= ul) ++d1;  // monotone in u: amortised ~gridDim / chunks-per-partition steps
      const unsigned long long pa = s_pst[r * 1025 + d1], pb = s_pst[r * 1025 + d1 + 1];
      const unsigned long long s0 = pa + (ul - cst[d1]) * TILE;
      U.src_k = (const T*)R.t1 + s0;
      U.src_p = nullptr;
      U.dst = R.t2;
      U.cur = R.cur2 + ((unsigned long long)d1 << P.b2);
      U.len = (uint32_t)min((unsigned long long)TILE, pb - s0);
    }
    return true;
  }
};

// element j of a thread in a unit: MODE 1 -> vector-friendly (4 / 2 consecutive per 16 B load),
// MODE 2 -> strided by NT
template <typename K, int MODE, int NT>
__device__ __forceinline__ uint32_t pass_elem(int j) {
  constexpr int VEC = 16 / sizeof(K);
  if (MODE == 1) return (uint32_t)(j / VEC) * NT * VEC + threadIdx.x * VEC + (j % VEC);
  return (uint32_t)j * NT + threadIdx.x;
}

template <typename K, int MODE, int NT, int ITEMS>
__device__ __forceinline__ void pass_load(const PassUnit<K>& U, K (&kk)[ITEMS], K (&pp)[ITEMS]) {
  using TT = Tup<K>;
  using T = typename TT::T;
  constexpr int TILE = NT * ITEMS;
  if (MODE == 1) {
    const K* keys = (const K*)U.src_k;
    const K* pays = (const K*)U.src_p;
    constexpr int VEC = 16 / sizeof(K);
    const bool vec_ok = (U.len == TILE) && ((reinterpret_cast<uintptr_t>(keys) & 15) == 0) &&
                        ((reinterpret_cast<uintptr_t>(pays) & 15) == 0);
    if (vec_ok) {
      #pragma unroll
      for (int j = 0; j < ITEMS / VEC; ++j) {
        const uint4 kv = __ldcs(reinterpret_cast<const uint4*>(keys) + j * NT + threadIdx.x);
        const uint4 pv = __ldcs(reinterpret_cast<const uint4*>(pays) + j * NT + threadIdx.x);
        const K* ke = reinterpret_cast<const K*>(&kv);
        const K* pe = reinterpret_cast<const K*>(&pv);
        #pragma unroll
        for (int t = 0; t < VEC; ++t) {
          kk[j * VEC + t] = ke[t];
          pp[j * VEC + t] = pe[t];
        }
      }
    } else {
      #pragma unroll
      for (int j = 0; j < ITEMS; ++j) {
        const uint32_t e = pass_elem<K, MODE, NT>(j);
        if (e < U.len) {
          kk[j] = keys[e];
          pp[j] = pays[e];
        }
      }
    }
  } else {
    const T* src = (const T*)U.src_k;
    #pragma unroll
    for (int j = 0; j < ITEMS; ++j) {
      const uint32_t e = pass_elem<K, MODE, NT>(j);
      if (e < U.len) {
        const T t = __ldcs(src + e);
        kk[j] = TT::key(t);
        pp[j] = TT::pay(t);
      }
    }
  }
}

template <typename K, int MODE, int NT, int ITEMS>
__global__ void __launch_bounds__(NT, 1) k_pass(Plan P, int fanout_bits) {
  using TT = Tup<K>;
  using T = typename TT::T;
  constexpr int TILE = NT * ITEMS;
  static_assert(NT >= 1024, "fan-out up to 2^10 needs one digit per thread");
  extern __shared__ __align__(16) unsigned char s_raw[];
  const uint32_t F = 1u << fanout_bits;
  T* s_buf = reinterpret_cast<T*>(s_raw);                                          // TILE tuples
  unsigned long long* s_gd = reinterpret_cast<unsigned long long*>(s_buf + TILE);  // F: run base - loc
  uint32_t* s_cnt = reinterpret_cast<uint32_t*>(s_gd + F);                         // F
  uint32_t* s_loc = s_cnt + F;                                                     // F
  __shared__ uint32_t s_tmp[NT / 32 + 1];
  __shared__ uint32_t s_cst[MODE == 2 ? 2 * 1025 : 1];
  __shared__ unsigned long long s_pst[MODE == 2 ? 2 * 1025 : 1];

  const uint32_t dmask = F - 1;
  const int dshift = (MODE == 1) ? 0 : P.b1;

  if (threadIdx.x < F) s_cnt[threadIdx.x] = 0;
  UnitWalker<K, MODE, TILE> W;
  W.rel = -1;
  W.d1 = 0;
  if (MODE == 1) {
    W.units0 = P.tiles1[0];
    W.units = W.units0 + P.tiles1[1];
  } else {
    for (uint32_t i = threadIdx.x; i <= (1u << P.b1); i += NT) {
      s_cst[i] = P.rel[0].cst[i];
      s_cst[1025 + i] = P.rel[1].cst[i];
      s_pst[i] = P.rel[0].off[(unsigned long long)i << P.b2];
      s_pst[1025 + i] = P.rel[1].off[(unsigned long long)i << P.b2];
    }
    W.units0 = P.rel[0].cst[1u << P.b1];
    W.units = W.units0 + P.rel[1].cst[1u << P.b1];
  }
  __syncthreads();

  PassUnit<K> U, Un;
  K kk[ITEMS], pp[ITEMS], kn[ITEMS], pn[ITEMS];
  unsigned long long u = blockIdx.x;
  bool have = W.get(P, u, U, s_cst, s_pst);
  if (have) pass_load<K, MODE, NT, ITEMS>(U, kn, pn);

  while (have) {
    #pragma unroll
    for (int j = 0; j < ITEMS; ++j) {
      kk[j] = kn[j];
      pp[j] = pn[j];
    }
    // prefetch the next unit (in flight across this unit's barriers)
    const bool have_next = W.get(P, u + gridDim.x, Un, s_cst, s_pst);
    if (have_next) pass_load<K, MODE, NT, ITEMS>(Un, kn, pn);

    // ---- rank ------------------------------------------------------------------------------
    uint32_t rk[ITEMS];
    #pragma unroll
    for (int j = 0; j < ITEMS; ++j)
      rk[j] = (pass_elem<K, MODE, NT>(j) < U.len) ? atomicAdd(&s_cnt[(uint32_t)(kk[j] >> dshift) & dmask], 1u)
                                                  : 0xffffffffu;
    __syncthreads();

    // ---- scan digit counts; issue the reservation atomic (result consumed after the shuffle)
    unsigned long long gres = 0;
    uint32_t myloc = 0;
    {
      const uint32_t d = threadIdx.x;
      const uint32_t c = (d < F) ? s_cnt[d] : 0u;
      uint32_t tot;
      myloc = block_exclusive_scan<NT>(c, s_tmp, &tot);
      if (d < F) {
        s_loc[d] = myloc;
        s_cnt[d] = 0;
        if (c) gres = atomicAdd(U.cur + d, (unsigned long long)c);
      }
    }
    __syncthreads();

    // ---- shuffle into digit order in shared memory -----------------------------------------
    #pragma unroll
    for (int j = 0; j < ITEMS; ++j)
      if (rk[j] != 0xffffffffu) s_buf[s_loc[(uint32_t)(kk[j] >> dshift) & dmask] + rk[j]] = TT::make(kk[j], pp[j]);
    if (threadIdx.x < F) s_gd[threadIdx.x] = gres - myloc;
    __syncthreads();

    // ---- stream runs out (consecutive threads -> consecutive addresses within a run) -------
    T* dst = (T*)U.dst;
    #pragma unroll
    for (int j = 0; j < ITEMS; ++j) {
      const uint32_t i = j * NT + threadIdx.x;
      if (i < U.len) {
        const T t = s_buf[i];
        __stcs(dst + (s_gd[(uint32_t)(TT::key(t) >> dshift) & dmask] + i), t);
      }
    }
    __syncthreads();  // s_buf / s_loc / s_gd are rewritten by the next unit
    U = Un;
    u += gridDim.x;
    have = have_next;
  }
}

}  // namespace hj
