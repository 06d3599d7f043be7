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
// block; or materialized: per round every thread counts its matches, a block scan
// gives exact offsets into a shared-memory output buffer, and a full buffer is flushed with one
// global atomicAdd on the output cursor and coalesced stores (the paper's buffered output,
// P:376-393, widened from a warp to a block so the global cursor sees one atomic per ~2K pairs).
#pragma once
#include "hj_common.cuh"
#include "hj_plan.cuh"

namespace hj {

constexpr uint32_t NIL16 = 0xffffu;

template <typename K, int NT, int SPT, bool MAT>
__global__ void __launch_bounds__(NT) k_join(Plan P, uint32_t ob_cap) {
  using TT = Tup<K>;
  using T = typename TT::T;
  extern __shared__ __align__(16) unsigned char s_raw[];
  const uint32_t nb = 1u << P.lg_nb;
  T* s_rt = reinterpret_cast<T*>(s_raw);                                    // CR tuples
  uint32_t* s_head = reinterpret_cast<uint32_t*>(s_rt + P.CR);              // nb
  uint16_t* s_next = reinterpret_cast<uint16_t*>(s_head + nb);              // CR
  K* s_obr = reinterpret_cast<K*>(reinterpret_cast<unsigned char*>(s_raw) +
                                  (((size_t)P.CR * sizeof(T) + (size_t)nb * 4 + (size_t)P.CR * 2 + 15) & ~(size_t)15));
  K* s_obs = s_obr + ob_cap;
  __shared__ uint32_t s_tmp[NT / 32 + 1];
  __shared__ uint32_t s_item, s_fill;
  __shared__ unsigned long long s_base;
  __shared__ unsigned long long s_red[2][NT / 32];

  const uint32_t np = 1u << P.B;
  const RelDev& RR = P.rel[0];
  const RelDev& SS = P.rel[1];
  const uint32_t total_items = P.ist[np];
  K* out_r = (K*)P.out_r;
  K* out_s = (K*)P.out_s;

  unsigned long long my_cnt = 0, my_chk = 0;
  if (MAT && threadIdx.x == 0) s_fill = 0;

  auto flush = [&]() {  // all threads; s_fill is block-uniform after a barrier
    __syncthreads();
    const uint32_t f = s_fill;
    if (f) {
      if (threadIdx.x == 0) s_base = atomicAdd(&P.results[RES_CURSOR], (unsigned long long)f);
      __syncthreads();
      const unsigned long long base = s_base;
      for (uint32_t i = threadIdx.x; i < f; i += NT) {
        if (base + i < P.out_cap) {
          __stcs(out_r + base + i, s_obr[i]);
          __stcs(out_s + base + i, s_obs[i]);
        }
      }
      __syncthreads();
      if (threadIdx.x == 0) s_fill = 0;
      __syncthreads();
    }
  };

  for (;;) {
    if (threadIdx.x == 0) s_item = atomicAdd(&P.counters[CNT_NEXT_ITEM], 1u);
    __syncthreads();
    const uint32_t item = s_item;
    if (item >= total_items) break;
    // item -> co-partition q: largest q with ist[q] <= item
    uint32_t lo = 0, hi = np;
    while (hi - lo > 1) {
      const uint32_t mid = (lo + hi) >> 1;
      if (P.ist[mid] <= item) lo = mid; else hi = mid;
    }
    const uint32_t q = lo;
    const unsigned long long r0 = RR.off[q], rn = RR.off[q + 1] - r0;
    const unsigned long long s0 = SS.off[q], sn = SS.off[q + 1] - s0;
    const unsigned long long nsch = (sn + P.CS - 1) / P.CS;
    const unsigned long long loc = item - P.ist[q];
    const unsigned long long rc = loc / nsch, sc = loc % nsch;
    const unsigned long long rb = r0 + rc * P.CR;
    const uint32_t nr = (uint32_t)min((unsigned long long)P.CR, rn - rc * P.CR);
    const unsigned long long sb = s0 + sc * P.CS;
    const unsigned long long se = sb + min((unsigned long long)P.CS, sn - sc * P.CS);

    // ---- build (a6) ----------------------------------------------------------------------
    const T* rsrc = (const T*)RR.t2 + rb;
    for (uint32_t i = threadIdx.x; i < nb; i += NT) s_head[i] = NIL16;
    for (uint32_t i = threadIdx.x; i < nr; i += NT) s_rt[i] = __ldcs(rsrc + i);
    __syncthreads();
    for (uint32_t i = threadIdx.x; i < nr; i += NT) {
      const uint32_t slot = slot_of(TT::key(s_rt[i]), P.B, P.lg_nb);
      s_next[i] = (uint16_t)atomicExch(&s_head[slot], i);
    }
    __syncthreads();

    // ---- probe (a7) + output (a8) --------------------------------------------------------
    const T* ssrc = (const T*)SS.t2;
    for (unsigned long long base = sb; base < se; base += (unsigned long long)NT * SPT) {
      K sk[SPT], sp[SPT];
      uint32_t m_t = 0;
      #pragma unroll
      for (int j = 0; j < SPT; ++j) {
        const unsigned long long s = base + (unsigned long long)j * NT + threadIdx.x;
        uint32_t idx = NIL16;
        if (s < se) {
          const T t = __ldcs(ssrc + s);
          sk[j] = TT::key(t);
          sp[j] = TT::pay(t);
          idx = s_head[slot_of(sk[j], P.B, P.lg_nb)];
        }
        while (idx != NIL16) {
          const T r = s_rt[idx];
          if (TT::key(r) == sk[j]) {
            ++m_t;
            my_chk += pair_sig((uint64_t)TT::pay(r), (uint64_t)sp[j]);
          }
          idx = s_next[idx];
        }
      }
      my_cnt += m_t;
      if (MAT) {
        uint32_t tot;
        uint32_t off = block_exclusive_scan<NT>(m_t, s_tmp, &tot);
        if (tot) {
          if (s_fill + tot > ob_cap) flush();
          const bool staged = tot <= ob_cap;
          unsigned long long gbase = 0;
          if (!staged) {  // more matches in one round than the buffer holds: write directly
            if (threadIdx.x == 0) s_base = atomicAdd(&P.results[RES_CURSOR], (unsigned long long)tot);
            __syncthreads();
            gbase = s_base;
          }
          const uint32_t f0 = s_fill;
          if (m_t) {
            #pragma unroll
            for (int j = 0; j < SPT; ++j) {
              const unsigned long long s = base + (unsigned long long)j * NT + threadIdx.x;
              if (s >= se) continue;
              uint32_t idx = s_head[slot_of(sk[j], P.B, P.lg_nb)];
              while (idx != NIL16) {
                const T r = s_rt[idx];
                if (TT::key(r) == sk[j]) {
                  if (staged) {
                    s_obr[f0 + off] = TT::pay(r);
                    s_obs[f0 + off] = sp[j];
                  } else if (gbase + off < P.out_cap) {
                    out_r[gbase + off] = TT::pay(r);
                    out_s[gbase + off] = sp[j];
                  }
                  ++off;
                }
                idx = s_next[idx];
              }
            }
          }
          __syncthreads();
          if (threadIdx.x == 0 && staged) s_fill = f0 + tot;
        }
        __syncthreads();
      }
    }
    __syncthreads();  // s_rt / s_head / s_item are rewritten by the next item
  }
  if (MAT) flush();

  // ---- aggregate: warp shuffle reduce, then one 64-bit atomic per block --------
  #pragma unroll
  for (int o = 16; o; o >>= 1) {
    my_cnt += __shfl_xor_sync(0xffffffffu, my_cnt, o);
    my_chk += __shfl_xor_sync(0xffffffffu, my_chk, o);
  }
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  if (lane == 0) {
    s_red[0][warp] = my_cnt;
    s_red[1][warp] = my_chk;
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

}  // namespace hj
