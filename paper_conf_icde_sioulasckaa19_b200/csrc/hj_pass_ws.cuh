// hj_pass_ws.cuh -- a3 / a4 (one radix-partition pass) as a warp-specialized pipeline.
//
// Same result as k_pass (hj_partition.cuh): every tuple of a unit is ranked within its digit with
// a shared-memory atomic, each digit's run is reserved in the output with one global atomic per
// (unit, digit), the unit is shuffled into digit order in shared memory and streamed out so
// consecutive threads write consecutive addresses of a run (P:142-148 coalescing; P:265-275
// metadata + shuffle space in shared memory). What changes is how an SM overlaps the steps: k_pass
// runs rank | write-out of the previous unit | shuffle with every warp of the block in lock step,
// so each SM's HBM traffic comes in bursts between block barriers (c3 pass 1: 0.95 ms, against
// 0.68 ms for the same access pattern with no shared-memory work, tools/microbench/mb_scatter.cu).
// Here one 1024-thread block per SM is three roles joined by mbarriers, over a ring of three
// shared-memory stages of one unit (tile) each:
//   producer (warp 31)    : unit descriptors; each unit's input copied into the next free stage
//                           by TMA bulk copies (cp.async.bulk: no registers, up to two units of
//                           input in flight per SM)
//   compute  (CW warps)   : stage -> registers, rank (shared atomics), scan + reserve (one global
//                           atomic per digit run), shuffle the registers back into the SAME stage
//                           in digit order (every read of the stage precedes a compute barrier)
//   writer   (31-CW warps): stage -> HBM in order, so consecutive threads write consecutive
//                           addresses of a run; then the stage is free for the producer
// so while the compute warps rank unit i, the writer streams unit i-1 and TMA fetches unit i+1:
// no role waits on another's shared-memory buffer except through the three-stage ring.
// Units whose input is ragged or not 16-byte aligned (the last unit of a relation, a piece whose
// aligned superset would leave the pass-1 data) are loaded by the compute warps from global.
// BC = true: the paper's bucket-chain partitioner (hj_bucket.cuh, NEXT-1): runs are reserved in
// the partitions' buckets (bc_reserve) instead of at histogram offsets, and pass 2's units are
// the pass-1 buckets cut into tiles (bucket at a time); the roles are unchanged.
#pragma once
#include "hj_common.cuh"
#include "hj_partition.cuh"
#include "hj_plan.cuh"

namespace hj {

constexpr int WS_NT = 1024;   // compute warps + writer warps + producer warp 31
constexpr int WS_MAXF = 512;  // fan-out bound (shared-memory budget)
constexpr int WS_NS = 3;      // stages

// Role split (HJ_OPT_PASS_WS): CW compute warps, 31 - CW writer warps; each compute thread ranks
// CIT tuples of a unit, so a unit (tile) has CW * 32 * CIT tuples (60 KB at CW = 20, the default).
template <typename K, int CW>
struct WsShape {
  static constexpr int CT = CW * 32, WT = (31 - CW) * 32;
  static constexpr int CIT = sizeof(K) == 4 ? (CW <= 16 ? 16 : CW <= 23 ? 12 : 8) : (CW <= 16 ? 8 : CW <= 23 ? 6 : 4);
  static constexpr int TILE = CT * CIT;
  static constexpr uint32_t STAGE = (uint32_t)TILE * 2 * sizeof(K) + 16;  // +16: aligned superset of AoS units
  static constexpr size_t smem(int fanout_bits) {  // stages + s_gd (3F u64) + s_cnt (F + 4) + s_loc (F)
    return WS_NS * (size_t)STAGE + ((size_t)1 << fanout_bits) * 32 + 16;
  }
};

__device__ __forceinline__ void mbar_arrive(unsigned long long* bar) {
  asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(bar)) : "memory");
}

struct WsUnit {
  const void* src_k;  // MODE 1: key column at the unit start; MODE 2: first AoS tuple
  const void* src_p;  // MODE 1: payload column at the unit start
  void* dst;          // output buffer (T1 or T2)
  unsigned long long* cur;  // reservation cursors (MODE 2: &cur2[D << b2])
  uint32_t len;
  uint32_t valid;
  uint32_t tma;    // input is in the stage (else: load from global)
  uint32_t shift;  // MODE 2: tuples between the stage start and the unit's first tuple
  uint32_t rel;    // bucket chains: relation, and the partition index of the unit's digit 0
  uint32_t pbase;
  uint32_t hot;    // the planner's skew hint for this unit's digits (RelDev::hot), HOT_NONE if none
};

template <typename K, int MODE, bool GD, int CW, bool BC = false>
__global__ void __launch_bounds__(WS_NT, 1) k_pass_ws(Plan P, int fanout_bits) {
  using TT = Tup<K>;
  using T = typename TT::T;
  using S = WsShape<K, CW>;
  constexpr int CT = S::CT, WT = S::WT, CIT = S::CIT, TILE = S::TILE;
  constexpr uint32_t STAGE = S::STAGE;
  constexpr int VEC = 16 / sizeof(K);
  static_assert(CIT % VEC == 0 && CIT % 2 == 0 && TILE < 65536, "tile shape");
  extern __shared__ __align__(128) unsigned char s_raw[];
  const uint32_t F = 1u << fanout_bits;
  unsigned long long* s_gd = reinterpret_cast<unsigned long long*>(s_raw + WS_NS * STAGE);  // 3 x F: run base - loc
  uint32_t* s_cnt = reinterpret_cast<uint32_t*>(s_gd + 3 * F);  // F + 1 (spare for ragged lanes)
  uint32_t* s_loc = s_cnt + F + 4;                              // F
  __shared__ __align__(8) unsigned long long s_full[WS_NS], s_empty[WS_NS], s_done[WS_NS];
  __shared__ WsUnit s_desc[4];
  __shared__ uint32_t s_wt[CT / 32];
  __shared__ uint32_t s_hot, s_hot_next;
  __shared__ uint32_t s_cst[MODE == 2 ? (BC ? 2 * BC_MAX_NB1 : 2 * 1025) : 1];
  __shared__ uint32_t s_hint2[MODE == 2 && !BC ? 2 * 1024 : 1];  // pass-2 skew hints per piece digit
  __shared__ uint32_t s_bfill[MODE == 2 && BC ? 2 * BC_MAX_NB1 : 1];  // bucket chains: pass-1 bucket fills
  __shared__ uint16_t s_bd[MODE == 2 && BC ? 2 * BC_MAX_NB1 : 1];     // and their partitions D
  __shared__ BcRel s_bc[BC ? 2 : 1];

  pdl_wait();
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  if (MODE == 2 && P.mode == PLAN_RECV && *(volatile const uint32_t*)&P.counters[CNT_BAD_COUNTS]) return;
  const uint32_t dsh = MODE == 1 ? 0u : (uint32_t)P.b1;
  const uint32_t dmask = MODE == 1 ? ((1u << P.b1) - 1) : ((1u << P.b2) - 1);
  const uint32_t gsh = (uint32_t)P.gsh, gmask = (1u << P.g) - 1, gup = (uint32_t)P.b1;
  auto digit = [=](K key) -> uint32_t {
    uint32_t d = (uint32_t)(key >> dsh) & dmask;
    if (MODE == 1 && GD) d |= ((uint32_t)(key >> gsh) & gmask) << gup;
    return d;
  };

  unsigned long long units0, units;
  if (BC) {
    if (threadIdx.x == 0) {
      s_bc[0] = P.bc_rel[0];
      s_bc[1] = P.bc_rel[1];
    }
    __syncthreads();
  }
  if (MODE == 1) {
    units0 = P.tiles1[0];
    units = units0 + P.tiles1[1];
  } else if (BC) {  // pass-1 buckets -> shared unit prefix (all threads)
    bc_pass2_units<WS_NT, TILE>(s_bc, P.counters, 1u << P.b1, s_cst, s_bfill, s_bd);
    __syncthreads();
    units0 = s_cst[2 * BC_MAX_NB1 - 3];
    units = s_cst[2 * BC_MAX_NB1 - 4];
  } else {
    const uint32_t npc = P.npieces();  // <= 1024
    for (uint32_t i = threadIdx.x; i <= npc; i += WS_NT) {
      s_cst[i] = P.rel[0].cst[i];
      s_cst[1025 + i] = P.rel[1].cst[i];
    }
    for (uint32_t i = threadIdx.x; i < (1u << P.pb()); i += WS_NT) {
      s_hint2[i] = P.rel[0].hot[1 + i];
      s_hint2[1024 + i] = P.rel[1].hot[1 + i];
    }
    units0 = P.skip_r ? 0ull : P.rel[0].cst[npc];
    units = units0 + P.rel[1].cst[npc];
  }
  if (threadIdx.x < F) s_cnt[threadIdx.x] = 0;
  if (threadIdx.x == 0) {
    s_hot = s_hot_next = 0xffffffffu;
    for (int s = 0; s < WS_NS; ++s) {
      mbar_init(&s_full[s], 1);         // producer (+ TMA bytes)
      mbar_init(&s_done[s], CT / 32);   // compute warps: the stage holds the shuffled unit
      mbar_init(&s_empty[s], WT / 32);  // writer warps: the stage is written out
    }
    fence_mbar_init();
  }
  __syncthreads();
  const unsigned long long G = gridDim.x;

  if (warp == 31) {
    // ---------------------------------------------------------------- producer ----------------
    if (lane != 0) return;
    const unsigned long long pend[2] = {MODE == 2 ? P.rel[0].pst[P.npieces()] : 0ull,
                                        MODE == 2 ? P.rel[1].pst[P.npieces()] : 0ull};
    const uint32_t hint1r = MODE == 1 && !BC ? P.rel[0].hot[0] : HOT_NONE;  // pass-1 skew hints
    const uint32_t hint1s = MODE == 1 && !BC ? P.rel[1].hot[0] : HOT_NONE;
    for (uint32_t i = 0;; ++i) {
      const uint32_t stage = i % WS_NS;
      // the descriptor is built before the wait for a free stage (its loads -- the unit search,
      // the piece bounds -- overlap the wait instead of delaying the copy); it is published
      // after the wait: slot i & 3 may still be read by the writer for unit i - 4 until then
      const unsigned long long u = blockIdx.x + (unsigned long long)i * G;
      WsUnit D;
      D.valid = u < units;
      D.tma = 0;
      D.shift = 0;
      D.pbase = 0;
      D.hot = HOT_NONE;
      if (D.valid) {
        const int r = u < units0 ? 0 : 1;
        const RelDev& R = P.rel[r];
        const unsigned long long ul = r ? u - units0 : u;
        D.rel = r;
        if (BC && MODE == 2) {  // unit -> (pass-1 bucket, tile) by binary search over the unit prefix
          const BcRel& Bc = s_bc[r];
          const uint32_t* cst = s_cst + r * BC_MAX_NB1;
          const uint32_t uc = (uint32_t)ul;
          uint32_t lo = 0, hi = s_cst[2 * BC_MAX_NB1 - 1 - r];  // buckets of r; largest with cst[b] <= uc
          while (hi - lo > 1) {
            const uint32_t mid = (lo + hi) >> 1;
            if (cst[mid] <= uc) lo = mid; else hi = mid;
          }
          const uint32_t k = uc - cst[lo];
          D.src_k = (const T*)Bc.pool1 + (unsigned long long)lo * Bc.bsz1 + (unsigned long long)k * TILE;
          D.src_p = nullptr;
          D.dst = Bc.pool2;
          D.pbase = (uint32_t)s_bd[r * BC_MAX_NB1 + lo] << P.b2;
          D.cur = nullptr;
          D.len = min((uint32_t)TILE, s_bfill[r * BC_MAX_NB1 + lo] - k * TILE);
          // bucket strides are tile multiples (16-byte aligned); the rounded-up copy stays inside
          // the bucket's stride (fill < cap + tile = bsz1)
          D.tma = 1;
        } else if (MODE == 1) {
          const unsigned long long s0 = ul * TILE;
          D.src_k = (const K*)R.keys + s0;
          D.src_p = (const K*)R.pays + s0;
          D.dst = BC ? P.bc_rel[r].pool1 : R.t1;
          D.cur = R.cur1;
          D.len = (uint32_t)min((unsigned long long)TILE, R.n - s0);
          D.tma = D.len == TILE && ((reinterpret_cast<uintptr_t>(D.src_k) | reinterpret_cast<uintptr_t>(D.src_p)) & 15) == 0;
          D.hot = r ? hint1s : hint1r;
        } else {
          const uint32_t* cst = s_cst + r * 1025;
          const uint32_t uc = (uint32_t)ul;
          uint32_t lo = 0, hi = P.npieces();  // largest piece with cst[piece] <= uc
          while (hi - lo > 1) {
            const uint32_t mid = (lo + hi) >> 1;
            if (cst[mid] <= uc) lo = mid; else hi = mid;
          }
          const unsigned long long pa = R.pst[lo], pb = R.pst[lo + 1];
          const unsigned long long s0 = pa + (unsigned long long)(uc - cst[lo]) * TILE;
          const uint32_t Dg = lo & ((1u << P.pb()) - 1);  // pass-1 digit of the piece
          D.src_k = (const T*)R.t1 + s0;
          D.src_p = nullptr;
          D.dst = R.t2;
          D.cur = R.cur2 + ((unsigned long long)Dg << P.b2);
          D.hot = s_hint2[r * 1024 + Dg];
          D.len = (uint32_t)min((unsigned long long)TILE, pb - s0);
          // the 16-byte aligned superset must stay inside the relation's pass-1 data
          const uintptr_t a = reinterpret_cast<uintptr_t>(D.src_k), a0 = a & ~(uintptr_t)15;
          const uintptr_t a1 = (a + (uintptr_t)D.len * sizeof(T) + 15) & ~(uintptr_t)15;
          D.tma = a1 <= reinterpret_cast<uintptr_t>((const T*)R.t1 + pend[r]);
          D.shift = (uint32_t)((a - a0) / sizeof(T));
        }
      }
      if (i >= WS_NS) mbar_wait(&s_empty[stage], ((i / WS_NS) - 1) & 1);  // unit i-3 written out
      s_desc[i & 3] = D;
      unsigned char* st = s_raw + stage * STAGE;
      if (D.valid && D.tma) {
        fence_proxy_async();  // earlier generic-proxy accesses of this stage precede the copy
        if (MODE == 1) {
          const uint32_t b = TILE * (uint32_t)sizeof(K);
          mbar_arrive_expect_tx(&s_full[stage], 2 * b);
          bulk_g2s(st, D.src_k, b, &s_full[stage]);
          bulk_g2s(st + b, D.src_p, b, &s_full[stage]);
        } else {
          const uintptr_t a = reinterpret_cast<uintptr_t>(D.src_k), a0 = a & ~(uintptr_t)15;
          const uint32_t b = (uint32_t)(((a + (uintptr_t)D.len * sizeof(T) - a0) + 15) & ~(uintptr_t)15);
          mbar_arrive_expect_tx(&s_full[stage], b);
          bulk_g2s(st, reinterpret_cast<const void*>(a0), b, &s_full[stage]);
        }
      } else {
        mbar_arrive(&s_full[stage]);  // descriptor only (the end marker, or a unit loaded from global)
      }
      if (!D.valid) return;
    }
  }

  if (warp >= CT / 32) {
    // ---------------------------------------------------------------- writer ------------------
    const uint32_t wt = threadIdx.x - CT;
    for (uint32_t i = 0;; ++i) {
      const uint32_t stage = i % WS_NS;
      mbar_wait(&s_done[stage], (i / WS_NS) & 1);  // the compute warps shuffled unit i (or ended)
      const WsUnit& D = s_desc[i & 3];
      if (!D.valid) return;
      T* dst = (T*)D.dst;
      const uint32_t len = D.len;
      const T* s_t = reinterpret_cast<const T*>(s_raw + stage * STAGE);
      const unsigned long long* gd = s_gd + (i % 3) * F;
      #pragma unroll 4
      for (uint32_t e = wt; e < len; e += WT) {
        const T t = s_t[e];
        __stcs(dst + (gd[digit(TT::key(t))] + e), t);
      }
      __syncwarp();
      if (lane == 0) mbar_arrive(&s_empty[stage]);
    }
  }

  // ------------------------------------------------------------------ compute -----------------
  const uint32_t nscan = F < 32 ? 32u : F;  // threads in the digit scan (whole warps)
  // element e of the unit held by thread (j, v): MODE 1 (j * CT + tid) * VEC + v (128-bit loads of
  // VEC keys / payloads), MODE 2 j * CT + tid
  auto elem = [&](int j) -> uint32_t {
    return MODE == 1 ? (uint32_t)((j / VEC) * CT + threadIdx.x) * VEC + (j % VEC) : (uint32_t)(j * CT + threadIdx.x);
  };
  for (uint32_t i = 0;; ++i) {
    const uint32_t stage = i % WS_NS;
    mbar_wait(&s_full[stage], (i / WS_NS) & 1);
    const WsUnit D = s_desc[i & 3];
    if (!D.valid) {
      __syncwarp();
      if (lane == 0) mbar_arrive(&s_done[stage]);  // end marker for the writer
      break;
    }
    const uint32_t ulen = D.len;
    const bool full = ulen == TILE;
    unsigned char* st = s_raw + stage * STAGE;
    K kk[CIT], pp[CIT];
    if (D.tma) {
      if (MODE == 1) {
        #pragma unroll
        for (int j = 0; j < CIT / VEC; ++j) {
          const uint4 kv = reinterpret_cast<const uint4*>(st)[j * CT + threadIdx.x];
          const uint4 pv = reinterpret_cast<const uint4*>(st + TILE * sizeof(K))[j * CT + threadIdx.x];
          const K* ke = reinterpret_cast<const K*>(&kv);
          const K* pe = reinterpret_cast<const K*>(&pv);
          #pragma unroll
          for (int v = 0; v < VEC; ++v) {
            kk[j * VEC + v] = ke[v];
            pp[j * VEC + v] = pe[v];
          }
        }
      } else {
        const T* src = reinterpret_cast<const T*>(st) + D.shift;
        #pragma unroll
        for (int j = 0; j < CIT; ++j) {
          if (full || elem(j) < ulen) {
            const T t = src[elem(j)];
            kk[j] = TT::key(t);
            pp[j] = TT::pay(t);
          }
        }
      }
    } else {
      #pragma unroll
      for (int j = 0; j < CIT; ++j) {
        const uint32_t e = elem(j);
        if (e < ulen) {
          if (MODE == 1) {
            kk[j] = ((const K*)D.src_k)[e];
            pp[j] = ((const K*)D.src_p)[e];
          } else {
            const T t = __ldcs((const T*)D.src_k + e);
            kk[j] = TT::key(t);
            pp[j] = TT::pay(t);
          }
        }
      }
    }

    // ---- rank (as k_pass: lanes on the predicted hot digit are ranked by ballot) -------------
    uint32_t rk[CIT / 2];
    // the hot digit: the planner's hint from the histogram (exact; pass 2 takes only the hint, as
    // its units change partition from one to the next), else in pass 1 the previous unit's
    // (bucket chains: no histogram)
    const uint32_t hot = D.hot != HOT_NONE ? D.hot : (MODE == 1 || BC ? s_hot : HOT_NONE);
    if (hot > F) {
      #pragma unroll
      for (int j = 0; j < CIT; ++j) {
        const uint32_t d = (full || elem(j) < ulen) ? digit(kk[j]) : F;
        const uint32_t r = atomicAdd(&s_cnt[d], 1u);
        if (j & 1) rk[j / 2] |= r << 16; else rk[j / 2] = r & 0xffffu;
      }
    } else {
      uint32_t hacc = 0, hbits = 0;
      const uint32_t lt = lanemask_lt();
      #pragma unroll
      for (int j = 0; j < CIT; ++j) {
        const uint32_t d = (full || elem(j) < ulen) ? digit(kk[j]) : F;
        const bool ih = d == hot;
        const uint32_t hm = __ballot_sync(0xffffffffu, ih);
        const uint32_t r = ih ? hacc + __popc(hm & lt) : atomicAdd(&s_cnt[d], 1u);
        hacc += __popc(hm);
        hbits |= (uint32_t)ih << j;
        if (j & 1) rk[j / 2] |= r << 16; else rk[j / 2] = r & 0xffffu;
      }
      if (hacc) {
        uint32_t base = 0;
        if (lane == 0) base = atomicAdd(&s_cnt[hot], hacc);
        base = __shfl_sync(0xffffffffu, base, 0);
        #pragma unroll
        for (int j = 0; j < CIT; ++j)
          if ((hbits >> j) & 1) rk[j / 2] += base << (16 * (j & 1));
      }
    }
    asm volatile("barrier.sync 1, %0;" ::"r"(CT) : "memory");  // every read of the stage is done

    // ---- scan + reserve (threads < F) ---------------------------------------------------------
    // each run's reservation atomic is issued here and its result stored after the shuffle, so
    // the global atomic's round trip overlaps the shuffle (the writer reads gd after s_done)
    unsigned long long* gd = s_gd + (i % 3) * F;
    unsigned long long rres = 0;
    uint32_t rloc = 0, rcnt = 0;
    bool rv = false;
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
      asm volatile("barrier.sync 2, %0;" ::"r"(nscan) : "memory");
      uint32_t base = 0;
      for (int w = 0; w < warp; ++w) base += s_wt[w];
      const uint32_t loc = base + x - c;
      if (d < F) {
        s_loc[d] = loc;
        s_cnt[d] = 0;
        if (c) {
          if (BC)  // the state's old value: finished (fast path or close / wait) after the shuffle
            rres = bc_reserve_issue<MODE>(&s_bc[D.rel], D.pbase + d, c);
          else
            rres = atomicAdd(D.cur + d, (unsigned long long)c);
          rloc = loc;
          rcnt = c;
          rv = true;
        }
        if (c > TILE / 4) atomicExch(&s_hot_next, d);  // predicts the next unit's hot digit
      }
    }
    asm volatile("barrier.sync 1, %0;" ::"r"(CT) : "memory");
    if (threadIdx.x == 0) {
      s_hot = s_hot_next;
      s_hot_next = 0xffffffffu;
    }
    // ---- shuffle the registers back into the stage, in digit order ---------------------------
    T* s_t = reinterpret_cast<T*>(st);
    #pragma unroll
    for (int j = 0; j < CIT; ++j)
      if (full || elem(j) < ulen)
        s_t[s_loc[digit(kk[j])] + ((rk[j / 2] >> (16 * (j & 1))) & 0xffffu)] = TT::make(kk[j], pp[j]);
    if (BC && rv)
      rres = bc_reserve_finish<MODE>(&s_bc[D.rel], &P.counters[(MODE == 1 ? CNT_BC_NB1 : CNT_BC_NB2) + D.rel],
                                     &P.results[RES_BC_OVERFLOW], D.pbase + threadIdx.x, rcnt, rres);
    if (rv) gd[threadIdx.x] = rres - rloc;
    __syncwarp();
    if (lane == 0) mbar_arrive(&s_done[stage]);  // unit i is ready for the writer
  }
}

}  // namespace hj
