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
#include "hj_bucket.cuh"
#include "hj_common.cuh"
#include "hj_plan.cuh"

namespace hj {

// ------------------------------------------------------------------------------------------
// a1: histogram. grid = (blocks_per_rel, 2). Each block counts a contiguous, 16-byte aligned
// range of one relation's keys in 2^qbits shared-memory counters indexed by the planner's
// q-order bin (smem atomics measured at ~6 tuples/clk/SM on B200, tools/microbench/mb_rank.cu),
// then merges non-zero counters with one global RED each (coalesced). For qbits > 15 (more than
// 128 KB of counters) SMEM = false counts with global atomics directly (correct, slower).
// ------------------------------------------------------------------------------------------
// Shared-memory counters, one 32-bit atomicAdd per key:
//   C32 = true : 2^qbits u32 counters (qbits <= 15, <= 128 KB)
//   C32 = false: 2^qbits u16 counters packed in pairs (qbits == 16, 128 KB). The increment that
//                takes a half from 0x7FFF to 0x8000 (seen in the atomic's return value) moves
//                0x8000 to the global counter and subtracts it from the half. The subtract is
//                issued as soon as that return arrives, long before another 0x8000 increments of
//                the same address can execute, so a half never passes 0xFFFF: no carry ever
//                reaches the neighbouring bin, and the flush adds each remainder.
template <bool C32>
__device__ __forceinline__ void hist_add(uint32_t* h, uint32_t bin, uint32_t* gcnt) {
  if (C32) {
    atomicAdd(&h[bin], 1u);
  } else {
    const uint32_t sh = (bin & 1) << 4;
    const uint32_t old = atomicAdd(&h[bin >> 1], 1u << sh);
    if (((old >> sh) & 0xffffu) == 0x7fffu) {
      atomicSub(&h[bin >> 1], 0x8000u << sh);
      atomicAdd(&gcnt[bin], 0x8000u);
    }
  }
}

template <typename K, bool SMEM, bool GD, bool C32 = true>
__global__ void __launch_bounds__(1024) k_hist(Plan P, uint32_t blocks_r) {
  extern __shared__ uint32_t s_hist[];
  const uint32_t np = 1u << P.qbits();
  const uint32_t nwords = C32 ? np : np / 2;
  if (SMEM) {
    for (uint32_t i = threadIdx.x; i < nwords; i += blockDim.x) s_hist[i] = 0;
  }
  __syncthreads();
  constexpr int VEC = 16 / sizeof(K);
  int rel = 0;
  auto add = [&](K key) {
    const uint32_t b = qbin<GD>(key, P);
    if (SMEM) hist_add<C32>(s_hist, b, P.rel[rel].cnt);
    else atomicAdd(&P.rel[rel].cnt[b], 1u);
  };
  // merge the shared q-histogram of relation r into the global one
  auto flush_q = [&](int r) {
    __syncthreads();
    for (uint32_t i = threadIdx.x; i < np; i += blockDim.x) {
      const uint32_t c = C32 ? s_hist[i] : ((s_hist[i >> 1] >> ((i & 1) << 4)) & 0xffffu);
      if (c) atomicAdd(&P.rel[r].cnt[i], c);
    }
  };
  auto count_range = [&](const K* keys, unsigned long long lo, unsigned long long hi) {
    if (lo >= hi) return;
    const bool aligned = ((reinterpret_cast<uintptr_t>(keys + lo) & 15) == 0);
    unsigned long long i = lo;
    if (aligned) {
      const unsigned long long nvec = (hi - lo) / VEC;
      const uint4* kv = reinterpret_cast<const uint4*>(keys + lo);
      constexpr int U = 4;  // 16 B loads per thread per batch
      // software-pipelined: batch k + 1 is loaded before batch k's atomics, so U loads per thread
      // stay in flight across the atomics (ptxas otherwise sinks each load to its first use,
      // leaving one 16-byte load per thread in flight: c3 0.196 -> 0.247 ms)
      unsigned long long v = threadIdx.x;
      const unsigned long long step = U * (unsigned long long)blockDim.x;
      if (v + (U - 1) * blockDim.x < nvec) {
        uint4 x[U];
        #pragma unroll
        for (int u = 0; u < U; ++u) x[u] = __ldcs(kv + v + u * blockDim.x);
        for (;;) {
          const unsigned long long vn = v + step;
          const bool more = vn + (U - 1) * blockDim.x < nvec;
          uint4 y[U];
          if (more) {
            #pragma unroll
            for (int u = 0; u < U; ++u) y[u] = __ldcs(kv + vn + u * blockDim.x);
          }
          #pragma unroll
          for (int u = 0; u < U; ++u) {
            const K* e = reinterpret_cast<const K*>(&x[u]);
            #pragma unroll
            for (int t = 0; t < VEC; ++t) add(e[t]);
          }
          v = vn;
          if (!more) break;
          #pragma unroll
          for (int u = 0; u < U; ++u) x[u] = y[u];
        }
      }
      for (; v < nvec; v += blockDim.x) {
        uint4 x = __ldcs(kv + v);
        const K* e = reinterpret_cast<const K*>(&x);
        #pragma unroll
        for (int t = 0; t < VEC; ++t) add(e[t]);
      }
      i = lo + nvec * VEC;
    }
    for (unsigned long long j = i + threadIdx.x; j < hi; j += blockDim.x) add(keys[j]);
  };
  // blocks [0, blocks_r) count R, the rest count S (split proportionally to |R| : |S|)
  rel = blockIdx.x < blocks_r ? 0 : 1;
  const unsigned long long n = P.rel[rel].n;
  const uint32_t nblk = rel ? gridDim.x - blocks_r : blocks_r;
  const uint32_t bid = rel ? blockIdx.x - blocks_r : blockIdx.x;
  unsigned long long per = (n + nblk - 1) / nblk;
  per = (per + VEC - 1) / VEC * VEC;
  const unsigned long long lo = (unsigned long long)bid * per;
  count_range((const K*)P.rel[rel].keys, lo, lo + per < n ? lo + per : n);
  if (SMEM) flush_q(rel);
}

// ------------------------------------------------------------------------------------------
// a1 on the exchange receiver: this rank's own histogram of the 2^B co-partitions of the AoS
// tuples it received (rel.t1, the first sum(prow) of them), in shared memory as k_hist (u32 bins
// up to 2^15, packed 16-bit bins at 2^16). After the exchange every key in the buffer belongs to
// this rank's 2^B co-partitions, so the counts are dense per bin; the senders then only count
// their (rank, d1) pieces (<= 2^10 bins) instead of 2^(g+B) bins in global memory.
// grid: blocks [0, blocks_r) count R, the rest S.
// ------------------------------------------------------------------------------------------
template <typename K, bool SMEM, bool C32>
__global__ void __launch_bounds__(1024) k_hist_recv(Plan P, uint32_t blocks_r) {
  using TT = Tup<K>;
  using T = typename TT::T;
  extern __shared__ uint32_t s_hist[];
  __shared__ unsigned long long s_tot;
  const uint32_t np = 1u << P.B;
  const uint32_t nwords = !SMEM ? 0u : C32 ? np : np / 2;
  const int rel = blockIdx.x < blocks_r ? 0 : 1;
  for (uint32_t i = threadIdx.x; i < nwords; i += blockDim.x) s_hist[i] = 0;
  if (threadIdx.x == 0) s_tot = 0;
  __syncthreads();
  {  // tuples received = sum of the piece rows (<= 1024 words)
    unsigned long long t = 0;
    for (uint32_t i = threadIdx.x; i < P.npieces(); i += blockDim.x) t += P.prow[rel][i];
    #pragma unroll
    for (int o = 16; o; o >>= 1) t += __shfl_xor_sync(0xffffffffu, t, o);
    if ((threadIdx.x & 31) == 0 && t) atomicAdd(&s_tot, t);
  }
  __syncthreads();
  const unsigned long long n = min(s_tot, P.rel[rel].n);
  const uint32_t nblk = rel ? gridDim.x - blocks_r : blocks_r;
  const uint32_t bid = rel ? blockIdx.x - blocks_r : blockIdx.x;
  const unsigned long long per = (n + nblk - 1) / nblk;
  const unsigned long long lo = min((unsigned long long)bid * per, n), hi = min(lo + per, n);
  const T* t1 = (const T*)P.rel[rel].t1;
  uint32_t* gcnt = P.rel[rel].cnt;
  auto add = [&](K key) {
    const uint32_t b = qbin<false>(key, P);
    if (!SMEM) atomicAdd(&gcnt[b], 1u);  // more than 2^16 bins: global atomics (correct, slower)
    else if (C32) atomicAdd(&s_hist[b], 1u);
    else hist_add<false>(s_hist, b, gcnt);
  };
  constexpr int U = 4;  // tuples per thread per batch (loaded before any atomic)
  unsigned long long i = lo + threadIdx.x;
  for (; i + (U - 1) * blockDim.x < hi; i += U * (unsigned long long)blockDim.x) {
    K k[U];
    #pragma unroll
    for (int u = 0; u < U; ++u) k[u] = TT::key(__ldcs(t1 + i + u * blockDim.x));
    #pragma unroll
    for (int u = 0; u < U; ++u) add(k[u]);
  }
  for (; i < hi; i += blockDim.x) add(TT::key(__ldcs(t1 + i)));
  if (!SMEM) return;
  __syncthreads();
  for (uint32_t q = threadIdx.x; q < np; q += blockDim.x) {
    const uint32_t c = C32 ? s_hist[q] : ((s_hist[q >> 1] >> ((q & 1) << 4)) & 0xffffu);
    if (c) atomicAdd(&gcnt[q], c);
  }
}

// ------------------------------------------------------------------------------------------
// a2 + a5: the planner. grid = ceil(2^qbits / 1024) blocks of 1024 threads.
//   off[q]  = exclusive scan over q of sum_s cnt[s][q]             (co-partition starts in T2)
//   cur2[q] = off[q]                                               (pass-2 reservation cursors)
//   pst[i]  = exclusive scan of piece sizes, i = (s, D)            (pass-2 input pieces in T1)
//   cur1[D] = pst[D] (one source)                                  (pass-1 reservation cursors)
//   cst[i]  = exclusive scan of ceil(|piece i| / C2)               (pass-2 chunk list)
//   ist[q]  = exclusive scan of items(q), items(q) = ceil(|R_q|/CR) * ceil(|S_q|/CS) if both
//             non-empty else 0                                     (join work list)
// Block b owns q in [1024 b, 1024 (b+1)), one q per thread, so every store is coalesced. Each
// block first sums all counts below its range itself (a redundant prefix: at most 2^qbits/1024
// independent loads per thread, L2-resident), then scans its own range. With several sources
// the blocks also sum piece sizes (a warp per piece). The last block (atomic ticket) scans the
// pieces.
// ------------------------------------------------------------------------------------------
__device__ __forceinline__ unsigned long long plan_items(const Plan& P, unsigned long long cr, unsigned long long cs) {
  if (!cr || !cs) return 0ull;
  if (cr <= P.CR && cs <= P.CS) return 1ull;  // the common case: no division (~20 instructions each)
  if (((cr | cs) >> 31) == 0)  // 32-bit division (a 64-bit one is ~10x the instructions)
    return (unsigned long long)(((uint32_t)cr + P.CR - 1) / P.CR) * (((uint32_t)cs + P.CS - 1) / P.CS);
  return ((cr + P.CR - 1) / P.CR) * ((cs + P.CS - 1) / P.CS);
}

__device__ __forceinline__ unsigned long long plan_count(const RelDev& R, int, uint32_t, uint32_t q) { return R.cnt[q]; }

// a co-partition is swapped when its R side needs several C_R chunks while its S side fits one:
// its items build on S and probe with R chunks of 2^lgCRp <= C_R tuples (a duplicate-heavy build side would
// otherwise walk chains of identical keys in single lanes)
__device__ __forceinline__ bool plan_swapped(const Plan& P, unsigned long long cr, unsigned long long cs) {
  return P.ist2 != nullptr && cr > P.CR && cs && cs <= P.CR;
}
__device__ __forceinline__ unsigned long long plan_items_swapped(const Plan& P, unsigned long long cr) {
  // probe chunks of 2^lgCRp <= C_R R tuples (k_join's claim_job<SWAP>)
  return (cr + (1ull << P.lgCRp) - 1) >> P.lgCRp;
}

// MS: several sources (exchange receiver); IT: join items (not on the exchange sender). Specialised so each launch runs (and fetches) only its own code.
template <bool MS, bool IT>
__global__ void __launch_bounds__(1024) k_plan(Plan P) {
  pdl_wait();
  constexpr int NT = 1024;
  __shared__ unsigned long long s_tmp6[6 * (NT / 32 + 1)];
  __shared__ bool s_last;
  const uint32_t np = 1u << P.qbits();
  const uint32_t b = blockIdx.x;
  const int nsrc = MS ? P.nsrc : 1;
  constexpr bool items = IT;
  // ---- prefix of everything below this block's range -------------------------------------
  unsigned long long sR = 0, sS = 0, sI = 0, sI2 = 0;
  // batches of 16 earlier blocks: all 32 count loads are issued before any is used (the loop is
  // latency-bound: one L2 round trip per batch instead of per block)
  for (uint32_t k0 = 0; k0 < b; k0 += 16) {
    uint32_t cr[16], cs[16];
    #pragma unroll
    for (int u = 0; u < 16; ++u) {
      const bool ok = k0 + u < b;
      cr[u] = ok ? (uint32_t)plan_count(P.rel[0], nsrc, np, (k0 + u) * NT + threadIdx.x) : 0u;
      cs[u] = ok ? (uint32_t)plan_count(P.rel[1], nsrc, np, (k0 + u) * NT + threadIdx.x) : 0u;
    }
    #pragma unroll
    for (int u = 0; u < 16; ++u) {
      sR += cr[u];
      sS += cs[u];
      if (items) {
        if (plan_swapped(P, cr[u], cs[u])) sI2 += plan_items_swapped(P, cr[u]);
        else sI += plan_items(P, cr[u], cs[u]);
      }
    }
  }
  // T2's 64-byte tails (the join's 16-byte aligned R copies may read into them; streaming S
  // chunks: T2 of R holds R, its tail is past R's end and stays)
  if (b == 0 && threadIdx.x < 32 && P.mode != PLAN_SEND) {
    const int r = threadIdx.x >> 4;
    if (P.rel[r].t2 && !(r == 0 && P.skip_r))
      reinterpret_cast<uint32_t*>(reinterpret_cast<char*>(P.rel[r].t2) + P.rel[r].n * (unsigned long long)P.tuple_bytes)[threadIdx.x & 15] = 0u;
  }
  // ---- own range ---------------------------------------------------------------------------
  const uint32_t q = b * NT + threadIdx.x;
  unsigned long long cr = 0, cs = 0;
  if (q < np) {
    cr = plan_count(P.rel[0], nsrc, np, q);
    cs = plan_count(P.rel[1], nsrc, np, q);
  }
  // the block totals of the prefix (reductions: exclusive scans whose totals are used) and this
  // range's three scans, all in ONE multi-value scan (one pair of barriers)
  // the normal and the swapped item counts share one scan value (low / high 32 bits: the item
  // totals are < 2^32, the join's item indices are u32)
  const bool swp = items && plan_swapped(P, cr, cs);
  const unsigned long long it2 = (items && !swp ? plan_items(P, cr, cs) : 0ull) |
                                 (swp ? plan_items_swapped(P, cr) : 0ull) << 32;
  unsigned long long v[6] = {sR, sS, sI | sI2 << 32, cr, cs, it2}, tt[6];
  block_exclusive_scan64xM<NT, 6>(v, s_tmp6, tt);
  const unsigned long long bR = tt[0], bS = tt[1], bI = tt[2] & 0xffffffffull, bI2 = tt[2] >> 32;
  const unsigned long long tR = tt[3], tS = tt[4], tI = tt[5] & 0xffffffffull, tI2 = tt[5] >> 32;
  const unsigned long long oR = bR + v[3], oS = bS + v[4];
  const unsigned long long oI = bI + (v[5] & 0xffffffffull), oI2 = bI2 + (v[5] >> 32);
  if (q < np) {
    P.rel[0].off[q] = oR;
    P.rel[0].cur2[q] = oR;
    P.rel[1].off[q] = oS;
    P.rel[1].cur2[q] = oS;
    if (items) P.ist[q] = (uint32_t)oI;
    if (items && P.ist2) P.ist2[q] = (uint32_t)oI2;
  }
  // ---- pass-2 skew hints: the d2 digit holding > 1/4 of its pass-1 partition ----------------
  // (a partition's 2^b2 bins lie in one block: b2 <= 10). k_pass_ws ranks that digit's tuples by
  // ballot instead of on one shared counter (c4: the Zipf keys' partitions).
  if (P.b2 > 0) {
    __shared__ unsigned long long s_psz[2][NT];  // sizes of this block's partitions (local index)
    __shared__ uint32_t s_hot2[2][NT];
    const uint32_t lp = threadIdx.x >> P.b2, d2 = threadIdx.x & ((1u << P.b2) - 1);
    if (threadIdx.x < (NT >> P.b2)) {  // this block's partitions
      s_psz[0][threadIdx.x] = s_psz[1][threadIdx.x] = 0ull;
      s_hot2[0][threadIdx.x] = s_hot2[1][threadIdx.x] = HOT_NONE;
    }
    __syncthreads();
    if (P.b2 >= 5) {  // a warp's 32 bins lie in one partition: one shared atomic per warp
      unsigned long long wr = cr, ws = cs;
      #pragma unroll
      for (int o = 16; o; o >>= 1) {
        wr += __shfl_xor_sync(0xffffffffu, wr, o);
        ws += __shfl_xor_sync(0xffffffffu, ws, o);
      }
      if ((threadIdx.x & 31) == 0) {
        if (wr) atomicAdd(&s_psz[0][lp], wr);
        if (ws) atomicAdd(&s_psz[1][lp], ws);
      }
    } else {
      if (cr) atomicAdd(&s_psz[0][lp], cr);
      if (cs) atomicAdd(&s_psz[1][lp], cs);
    }
    __syncthreads();
    if (cr && 4 * cr > s_psz[0][lp]) s_hot2[0][lp] = d2;  // at most three digits qualify; any one wins
    if (cs && 4 * cs > s_psz[1][lp]) s_hot2[1][lp] = d2;
    __syncthreads();
    if (q < np && d2 == 0) {
      P.rel[0].hot[1 + (q >> P.b2)] = s_hot2[0][lp];
      P.rel[1].hot[1 + (q >> P.b2)] = s_hot2[1][lp];
    }
  }
  if (b == gridDim.x - 1 && threadIdx.x == 0) {
    P.rel[0].off[np] = bR + tR;
    P.rel[1].off[np] = bS + tS;
    bool bad = false;
    if (P.mode == PLAN_RECV) {  // received count rows must not describe more tuples than the buffers hold
      bad = bR + tR > P.rel[0].n || bS + tS > P.rel[1].n;
      if (bad) P.counters[CNT_BAD_COUNTS] = 1u;  // pass 2 and the join then do nothing
    }
    if (items) P.ist[np] = bad ? 0u : (uint32_t)(bI + tI);
    if (items && P.ist2) P.ist2[np] = bad ? 0u : (uint32_t)(bI2 + tI2);
  }
  // ---- last block: piece starts, pass-1 cursors, pass-2 chunk lists (npieces <= 1024) ------
  __threadfence();
  __syncthreads();
  if (threadIdx.x == 0) s_last = atomicAdd(&P.counters[CNT_PLAN_DONE], 1u) == gridDim.x - 1;
  __syncthreads();
  if (!s_last) return;
  __threadfence();
  const uint32_t npieces = P.npieces();
  const int b2 = P.b2;
  const uint32_t i = threadIdx.x;
  unsigned long long pv[4], ptt[4];  // (piece size, its pass-2 chunks) of R, then of S
  #pragma unroll
  for (int rel = 0; rel < 2; ++rel) {
    const RelDev& R = P.rel[rel];
    unsigned long long sz = 0;
    if (i < npieces) {
      if (nsrc == 1)
        sz = __ldcg(&R.off[(unsigned long long)(i + 1) << b2]) - __ldcg(&R.off[(unsigned long long)i << b2]);
      else
        sz = P.prow[rel][i];  // exchange receiver: piece i = (source i >> pb, digit) as sent
    }
    pv[2 * rel] = sz;
    pv[2 * rel + 1] = (sz + P.C2 - 1) / P.C2;
  }
  if (P.mode == PLAN_RECV) {
    // the pieces of pass-1 digit D (one per source) must hold exactly what this rank's own
    // histogram counted in D's co-partitions; else the rows describe other tuples than the
    // buffers hold (pass 2 and the join then do nothing, hj_join_received fails)
    const uint32_t F1 = 1u << P.pb();
    for (int rel = 0; rel < 2 && i < F1; ++rel) {
      unsigned long long sent = 0;
      for (int sr = 0; sr < nsrc; ++sr) sent += P.prow[rel][(size_t)sr * F1 + i];
      const RelDev& R = P.rel[rel];
      const unsigned long long got = __ldcg(&R.off[(unsigned long long)(i + 1) << b2]) - __ldcg(&R.off[(unsigned long long)i << b2]);
      if (sent != got) {
        P.counters[CNT_BAD_COUNTS] = 1u;
        if (rel == 0) {
          P.ist[1u << P.B] = 0u;
          if (P.ist2) P.ist2[1u << P.B] = 0u;
        }
      }
    }
  }
  // pass-1 skew hints: the pass-1 digit holding > 1/4 of the relation (one source only: the
  // receiver runs no pass 1); the defaults are written before the scan, whose barriers order them
  // before the hints written after it
  bool hot1[2];
  #pragma unroll
  for (int rel = 0; rel < 2; ++rel) hot1[rel] = nsrc == 1 && i < npieces && pv[2 * rel] && 4 * pv[2 * rel] > P.rel[rel].n;
  if (i == 0) P.rel[0].hot[0] = P.rel[1].hot[0] = HOT_NONE;
  block_exclusive_scan64xM<NT, 4>(pv, s_tmp6, ptt);  // pv becomes the exclusive prefix
  #pragma unroll
  for (int rel = 0; rel < 2; ++rel) {
    const RelDev& R = P.rel[rel];
    if (hot1[rel]) R.hot[0] = i;
    if (i < npieces) {
      R.pst[i] = pv[2 * rel];
      R.cst[i] = (uint32_t)pv[2 * rel + 1];
      if (nsrc == 1) R.cur1[i] = pv[2 * rel];
    }
    if (i == 0) {
      R.pst[npieces] = ptt[2 * rel];
      R.cst[npieces] = (uint32_t)ptt[2 * rel + 1];
    }
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
struct __align__(16) PassUnit {
  const void* src_k;  // MODE 1: key column at the unit start; MODE 2: first AoS tuple of the unit
  const void* src_p;  // MODE 1: payload column at the unit start
  void* dst;          // output buffer (T1 or T2) of the unit's relation
  unsigned long long* cur;  // reservation cursors: cur1 (MODE 1) or &cur2[d1 << b2] (MODE 2)
  uint32_t len;
  uint32_t valid;
  uint32_t rel;    // bucket chains (BC): relation and first partition index of the unit's digits
  uint32_t pbase;
};

// Unit u (round-robin: u = blockIdx.x + k * gridDim.x) -> its descriptor. MODE 2 maps the chunk
// to its piece by binary search in the shared-memory chunk prefix (stateless: no registers live
// across the unit loop).
template <typename K, int MODE, int TILE, bool BC = false>
struct UnitWalker {
  unsigned long long units0, units;
  __device__ __forceinline__ bool get(const Plan& P, unsigned long long u, PassUnit<K>& U, const uint32_t* s_cst,
                                      const unsigned long long* s_pst, const uint32_t* s_bfill = nullptr,
                                      const uint16_t* s_bd = nullptr) const {
    using T = typename Tup<K>::T;
    // bucket-chain pass 2 keeps its unit counts in shared memory (spare top slots of s_cst):
    // no registers live across k_pass's tile loop
    const unsigned long long n0 = (BC && MODE == 2) ? s_cst[2 * BC_MAX_NB1 - 3] : units0;
    const unsigned long long nn = (BC && MODE == 2) ? s_cst[2 * BC_MAX_NB1 - 4] : units;
    U.valid = u < nn;
    if (!U.valid) return false;
    const int r = (u < n0) ? 0 : 1;
    const unsigned long long ul = r ? u - n0 : u;
    const RelDev& R = P.rel[r];
    U.rel = r;
    U.pbase = 0;
    if (BC) {  // bucket chains: pass 1 as below into the pass-1 pool; pass 2 = one bucket unit
      const BcRel& Bc = P.bc_rel[r];
      if (MODE == 1) {
        const unsigned long long s0 = ul * TILE;
        U.src_k = (const K*)R.keys + s0;
        U.src_p = (const K*)R.pays + s0;
        U.dst = Bc.pool1;
        U.cur = Bc.st1;
        U.len = (uint32_t)min((unsigned long long)TILE, R.n - s0);
      } else {  // unit -> (pass-1 bucket, tile) by binary search over the shared unit prefix
        const uint32_t* cst = s_cst + r * BC_MAX_NB1;
        const uint32_t uc = (uint32_t)ul;
        uint32_t lo = 0, hi = s_cst[2 * BC_MAX_NB1 - 1 - r];  // buckets of r; largest with cst[b] <= uc
        while (hi - lo > 1) {
          const uint32_t mid = (lo + hi) >> 1;
          if (cst[mid] <= uc) lo = mid; else hi = mid;
        }
        const uint32_t k = uc - cst[lo];
        U.src_k = (const T*)Bc.pool1 + (unsigned long long)lo * Bc.bsz1 + (unsigned long long)k * TILE;
        U.src_p = nullptr;
        U.dst = Bc.pool2;
        U.pbase = (uint32_t)s_bd[r * BC_MAX_NB1 + lo] << P.b2;
        U.cur = Bc.st2 + U.pbase;
        U.len = min((uint32_t)TILE, s_bfill[r * BC_MAX_NB1 + lo] - k * TILE);
      }
      return true;
    }
    if (MODE == 1) {
      const unsigned long long s0 = ul * TILE;
      U.src_k = (const K*)R.keys + s0;
      U.src_p = (const K*)R.pays + s0;
      U.dst = R.t1;
      U.cur = R.cur1;
      U.len = (uint32_t)min((unsigned long long)TILE, R.n - s0);
    } else {
      const uint32_t* cst = s_cst + r * 1025;
      const uint32_t uc = (uint32_t)ul;
      uint32_t lo = 0, hi = P.npieces();  // largest piece with cst[piece] <= uc
      while (hi - lo > 1) {
        const uint32_t mid = (lo + hi) >> 1;
        if (cst[mid] <= uc) lo = mid; else hi = mid;
      }
      const unsigned long long pa = s_pst[r * 1025 + lo], pb = s_pst[r * 1025 + lo + 1];
      const unsigned long long s0 = pa + (unsigned long long)(uc - cst[lo]) * TILE;
      const uint32_t D = lo & ((1u << P.pb()) - 1);  // pass-1 digit of the piece
      U.src_k = (const T*)R.t1 + s0;
      U.src_p = nullptr;
      U.dst = R.t2;
      U.cur = R.cur2 + ((unsigned long long)D << P.b2);
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

// Two-barrier software pipeline per unit i (one block of NT threads):
//   phase 1  rank unit i (smem atomics)                                            | barrier
//   phase 2  all threads: write unit i-1 out of s_buf (its run bases in s_gd[(i-1)&1]);
//            threads d < F additionally scan unit i's digit counts (named barrier among them),
//            reserve each run with one global atomic and store base - loc in s_gd[i&1]  | barrier
//   phase 3  shuffle unit i into digit order in s_buf
// so each reservation atomic's latency overlaps the previous unit's write-out.
// Bucket chains, pass 2 prologue: pass-1 buckets -> shared unit prefix (the bucket-at-a-time
// unit list). Each bucket's fill (its partition's state if it is the current bucket,
// else recorded by its closer), partition and pass-2 tiles, scanned over the buckets (<= 1.5 x
// 2^b1 + 1 per relation). Not inlined: keeps its temporaries out of k_pass's register budget.
template <int NT, int TILE>
__device__ __noinline__ void bc_pass2_units(const BcRel* s_bc, const uint32_t* counters, uint32_t F1, uint32_t* s_cst,
                                            uint32_t* s_bfill, uint16_t* s_bd) {
  __shared__ unsigned long long s_scan[NT / 32 + 1];
  unsigned long long tot[2];
  for (int r = 0; r < 2; ++r) {
    const BcRel& Bc = s_bc[r];
    const uint32_t nb = min(F1 + counters[CNT_BC_NB1 + r], Bc.nbmax1);
    const uint32_t per = (nb + NT - 1) / NT, b0 = threadIdx.x * per, b1 = min(b0 + per, nb);
    unsigned long long mine = 0;
    for (uint32_t b = b0; b < b1; ++b) {
      const uint32_t p = b < F1 ? b : Bc.part1[b];
      const unsigned long long st = Bc.st1[p];
      const uint32_t j = (uint32_t)(st >> 32);
      const uint32_t f = (j ? F1 + j - 1 : p) == b ? (uint32_t)st : Bc.fill1[b];
      s_bfill[r * BC_MAX_NB1 + b] = f;
      s_bd[r * BC_MAX_NB1 + b] = (uint16_t)p;
      mine += (f + TILE - 1) / TILE;
    }
    unsigned long long u = block_exclusive_scan64<NT>(mine, s_scan, &tot[r]);
    for (uint32_t b = b0; b < b1; ++b) {
      s_cst[r * BC_MAX_NB1 + b] = (uint32_t)u;
      u += (s_bfill[r * BC_MAX_NB1 + b] + TILE - 1) / TILE;
    }
    if (threadIdx.x == 0) {
      s_cst[r * BC_MAX_NB1 + nb] = (uint32_t)tot[r];
      s_cst[2 * BC_MAX_NB1 - 1 - r] = nb;  // bucket counts in the two spare top slots
    }
  }
  if (threadIdx.x == 0) {
    s_cst[2 * BC_MAX_NB1 - 3] = (uint32_t)tot[0];
    s_cst[2 * BC_MAX_NB1 - 4] = (uint32_t)(tot[0] + tot[1]);
  }
}

// RPF: the next unit's tuples are prefetched into registers during the current unit (default);
// RPF = false loads each unit at the top of its iteration (half the data registers: twice the
// tuples per thread at the same register budget, for two blocks per SM whose barriers overlap).
template <typename K, int MODE, int NT, int ITEMS, bool GD, bool BC = false, bool RPF = true>
__device__ __forceinline__ void pass_body(const Plan& P, int fanout_bits) {
  using TT = Tup<K>;
  using T = typename TT::T;
  constexpr int TILE = NT * ITEMS;
  static_assert(NT == 512 || NT == 1024, "block size");  // the launcher guarantees fan-out <= NT
  static_assert(TILE <= 65536 && ITEMS % 2 == 0, "16-bit packed ranks");
  extern __shared__ __align__(16) unsigned char s_raw[];
  const uint32_t F = 1u << fanout_bits;
  T* s_buf = reinterpret_cast<T*>(s_raw);                                          // TILE tuples
  unsigned long long* s_gd = reinterpret_cast<unsigned long long*>(s_buf + TILE);  // 2 x F: run base - loc
  uint32_t* s_cnt = reinterpret_cast<uint32_t*>(s_gd + 2 * F);                     // F + 1 (spare)
  uint32_t* s_loc = s_cnt + F + 4;                                                 // F
  __shared__ uint32_t s_wt[NT / 32];
  __shared__ uint32_t s_hot, s_hot_next;
  __shared__ uint32_t s_cst[MODE == 2 ? 2 * (BC ? BC_MAX_NB1 : 1025) : 1];
  __shared__ unsigned long long s_pst[MODE == 2 && !BC ? 2 * 1025 : 1];
  __shared__ uint32_t s_bfill[MODE == 2 && BC ? 2 * BC_MAX_NB1 : 1];  // bucket chains: pass-1 bucket fills
  __shared__ uint16_t s_bd[MODE == 2 && BC ? 2 * BC_MAX_NB1 : 1];     // and their partitions D
  __shared__ BcRel s_bc[BC ? 2 : 1];                                  // bucket chains: the plan's BcRel

  // digit of a key in this pass: D (pass 1, possibly widened by rank bits) or d2 (pass 2);
  // shifts and masks live in registers (not re-read from the parameter struct per tuple)
  const uint32_t dsh = MODE == 1 ? 0u : (uint32_t)P.b1;
  const uint32_t dmask = MODE == 1 ? ((1u << P.b1) - 1) : ((1u << P.b2) - 1);
  const uint32_t gsh = (uint32_t)P.gsh, gmask = (1u << P.g) - 1, gup = (uint32_t)P.b1;
  auto digit = [=](K key) -> uint32_t {
    uint32_t d = (uint32_t)(key >> dsh) & dmask;
    if (MODE == 1 && GD) d |= ((uint32_t)(key >> gsh) & gmask) << gup;
    return d;
  };
  const uint32_t nscan = F < 32 ? 32u : F;  // threads in the digit scan (whole warps)
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  // the exchange receiver's planner rejected the received count rows: nothing to do (block-uniform)
  if (MODE == 2 && !BC && P.mode == PLAN_RECV && *(volatile const uint32_t*)&P.counters[CNT_BAD_COUNTS]) return;

  if (threadIdx.x < F) s_cnt[threadIdx.x] = 0;
  if (threadIdx.x == 0) s_hot = s_hot_next = 0xffffffffu;
  UnitWalker<K, MODE, TILE, BC> W;
  if (MODE == 1) {
    W.units0 = P.tiles1[0];
    W.units = W.units0 + P.tiles1[1];
  } else if (BC) {
    if (threadIdx.x == 0) {
      s_bc[0] = P.bc_rel[0];
      s_bc[1] = P.bc_rel[1];
    }
    __syncthreads();
    bc_pass2_units<NT, TILE>(s_bc, P.counters, 1u << P.b1, s_cst, s_bfill, s_bd);
    W.units0 = W.units = 0;  // unused: get() reads the counts from s_cst
  } else {
    const uint32_t npc = P.npieces();  // <= 1024
    for (uint32_t i = threadIdx.x; i <= npc; i += NT) {
      s_cst[i] = P.rel[0].cst[i];
      s_cst[1025 + i] = P.rel[1].cst[i];
      s_pst[i] = P.rel[0].pst[i];
      s_pst[1025 + i] = P.rel[1].pst[i];
    }
    W.units0 = P.skip_r ? 0ull : P.rel[0].cst[npc];
    W.units = W.units0 + P.rel[1].cst[npc];
  }
  __syncthreads();

  // unit descriptors live in a 3-slot shared ring: one thread computes unit i+2 during unit i's
  // phase 2 (slot (i+2) % 3 held unit i-1, whose fields were copied to registers already)
  __shared__ PassUnit<K> s_desc[3];
  if (BC && MODE == 1 && threadIdx.x == 0) {
    s_bc[0] = P.bc_rel[0];
    s_bc[1] = P.bc_rel[1];
  }
  const unsigned long long G = gridDim.x;
  if (threadIdx.x == NT - 1) {
    W.get(P, blockIdx.x, s_desc[0], s_cst, s_pst, s_bfill, s_bd);
    W.get(P, blockIdx.x + G, s_desc[1], s_cst, s_pst, s_bfill, s_bd);
  }
  __syncthreads();
  T* prev_dst = nullptr;  // unit i-1 awaiting write-out
  uint32_t prev_len = 0;
  K kk[ITEMS], pp[ITEMS], kn[RPF ? ITEMS : 1], pn[RPF ? ITEMS : 1];
  unsigned long long u = blockIdx.x;
  if constexpr (RPF) {
    if (s_desc[0].valid) pass_load<K, MODE, NT, ITEMS>(s_desc[0], kn, pn);
  }
  uint32_t it = 0, slot = 0;

  auto write_out = [&](const unsigned long long* gd) {
    if (prev_len == TILE) {
      #pragma unroll
      for (int j = 0; j < ITEMS; ++j) {
        const uint32_t i = j * NT + threadIdx.x;
        const T t = s_buf[i];
        __stcs(prev_dst + (gd[digit(TT::key(t))] + i), t);
      }
    } else {
      #pragma unroll
      for (int j = 0; j < ITEMS; ++j) {
        const uint32_t i = j * NT + threadIdx.x;
        if (i < prev_len) {
          const T t = s_buf[i];
          __stcs(prev_dst + (gd[digit(TT::key(t))] + i), t);
        }
      }
    }
  };

  while (s_desc[slot].valid) {
    const uint32_t nslot = slot == 2 ? 0 : slot + 1;
    if constexpr (RPF) {
      #pragma unroll
      for (int j = 0; j < ITEMS; ++j) {
        kk[j] = kn[j];
        pp[j] = pn[j];
      }
    } else {
      pass_load<K, MODE, NT, ITEMS>(s_desc[slot], kk, pp);
    }
    // prefetch the next unit (in flight across this unit's barriers)
    if constexpr (RPF) {
      if (s_desc[nslot].valid) pass_load<K, MODE, NT, ITEMS>(s_desc[nslot], kn, pn);
    }

    // ---- phase 1: rank ------------------------------------------------------------------------
    // elements past the unit's end count into the spare counter s_cnt[F] (no branches)
    uint32_t rk[ITEMS / 2];  // ranks < TILE <= 2^16, two per register
    const uint32_t ulen = s_desc[slot].len;
    const bool full = ulen == TILE;
    const uint32_t hot = s_hot;  // digit holding > 1/4 of the previous unit, or none (> F)
    if (hot > F) {
      #pragma unroll
      for (int j = 0; j < ITEMS; ++j) {
        const uint32_t d = (full || pass_elem<K, MODE, NT>(j) < ulen) ? digit(kk[j]) : F;
        const uint32_t r = atomicAdd(&s_cnt[d], 1u);
        if (j & 1) rk[j / 2] |= r << 16; else rk[j / 2] = r & 0xffffu;
      }
    } else {
      // skew: lanes on the hot digit do not touch its shared counter item by item (same-address
      // atomics serialise); they are ranked inside the warp by ballot + popc, the warp reserves
      // its hot total with ONE atomic after all ITEMS and adds that base to its hot items' ranks
      // (Zipf probe sides). Branch-free per item: the other lanes' atomic is
      // the only per-item shared-memory access.
      uint32_t hacc = 0, hbits = 0;  // this warp's hot items so far; this thread's hot items (bit j)
      const uint32_t lt = lanemask_lt();
      #pragma unroll
      for (int j = 0; j < ITEMS; ++j) {
        const uint32_t d = (full || pass_elem<K, MODE, NT>(j) < ulen) ? digit(kk[j]) : F;
        const bool ih = d == hot;
        const uint32_t hm = __ballot_sync(0xffffffffu, ih);
        const uint32_t r = ih ? hacc + __popc(hm & lt) : atomicAdd(&s_cnt[d], 1u);
        hacc += __popc(hm);
        hbits |= (uint32_t)ih << j;
        if (j & 1) rk[j / 2] |= r << 16; else rk[j / 2] = r & 0xffffu;
      }
      if (hacc) {  // warp-uniform
        uint32_t base = 0;
        if (lane == 0) base = atomicAdd(&s_cnt[hot], hacc);
        base = __shfl_sync(0xffffffffu, base, 0);
        #pragma unroll
        for (int j = 0; j < ITEMS; ++j)
          if ((hbits >> j) & 1) rk[j / 2] += base << (16 * (j & 1));
      }
    }
    __syncthreads();

    // ---- phase 2: scan + reserve unit i (threads < F) | write unit i-1 out (all) ---------------
    unsigned long long* gd = s_gd + (it & 1) * F;
    if (threadIdx.x < nscan) {
      const uint32_t d = threadIdx.x;
      const uint32_t c = d < F ? s_cnt[d] : 0u;
      uint32_t x = c;
      #pragma unroll
      for (int o = 1; o < 32; o <<= 1) {
        const uint32_t y = __shfl_up_sync(0xffffffffu, x, o);
        if (lane >= o) x += y;
      }
      if (lane == 31) s_wt[warp] = x;
      asm volatile("barrier.sync 1, %0;" ::"r"(nscan) : "memory");
      uint32_t base = 0;
      for (int w = 0; w < warp; ++w) base += s_wt[w];
      const uint32_t loc = base + x - c;
      if (d < F) {
        s_loc[d] = loc;
        s_cnt[d] = 0;
        if (c) {
          if (BC) {
            const int r = (int)s_desc[slot].rel;
            gd[d] = bc_reserve<MODE>(&s_bc[r], &P.counters[(MODE == 1 ? CNT_BC_NB1 : CNT_BC_NB2) + r],
                               &P.results[RES_BC_OVERFLOW], s_desc[slot].pbase + d, c) - loc;
          }
          else gd[d] = atomicAdd(s_desc[slot].cur + d, (unsigned long long)c) - loc;
        }
        if (c > TILE / 4) atomicExch(&s_hot_next, d);  // predicts the next unit's hot digit (any one)
      }
    }
    if (threadIdx.x == NT - 1) {  // publish unit i+2
      PassUnit<K>& Dn = s_desc[nslot == 2 ? 0 : nslot + 1];
      W.get(P, u + 2 * G, Dn, s_cst, s_pst, s_bfill, s_bd);
      if (P.pass_l2pf && Dn.valid && Dn.len) {  // unit i+2's input -> L2 (its register loads come next iteration)
        const uint32_t bytes = MODE == 1 ? Dn.len * (uint32_t)sizeof(K) : Dn.len * (uint32_t)sizeof(T);
        const uintptr_t a = reinterpret_cast<uintptr_t>(Dn.src_k);
        if (((a | bytes) & 15) == 0) {
          bulk_prefetch_l2(Dn.src_k, bytes);
          if (MODE == 1 && (reinterpret_cast<uintptr_t>(Dn.src_p) & 15) == 0) bulk_prefetch_l2(Dn.src_p, bytes);
        }
      }
    }
    write_out(s_gd + ((it + 1) & 1) * F);
    __syncthreads();

    // ---- phase 3: shuffle unit i into digit order in shared memory -----------------------------
    if (threadIdx.x == 0) {  // read by the next unit's phase 1 (after this thread's own reads)
      s_hot = s_hot_next;
      s_hot_next = 0xffffffffu;
    }
    #pragma unroll
    for (int j = 0; j < ITEMS; ++j)
      if (full || pass_elem<K, MODE, NT>(j) < ulen)
        s_buf[s_loc[digit(kk[j])] + ((rk[j / 2] >> (16 * (j & 1))) & 0xffffu)] = TT::make(kk[j], pp[j]);
    // (no barrier: the next unit's phase 1 touches only s_cnt; its phase 2 reads s_buf / s_gd
    //  after the next phase-1 barrier)
    prev_dst = (T*)s_desc[slot].dst;
    prev_len = ulen;
    u += G;
    slot = nslot;
    ++it;
  }
  __syncthreads();
  write_out(s_gd + ((it + 1) & 1) * F);  // the last unit (it was incremented past it)
}

template <typename K, int MODE, int NT, int ITEMS, bool GD, bool BC = false, bool RPF = true>
__global__ void __launch_bounds__(NT, 1024 / NT) k_pass(Plan P, int fanout_bits) {
  pass_body<K, MODE, NT, ITEMS, GD, BC, RPF>(P, fanout_bits);
}

}  // namespace hj
