// hj_fused.cuh -- pass 2 (a4) and the co-partition join (a5-a8) in ONE persistent kernel, so
// the co-partitions pass 2 writes are joined while they are still in B200's 126 MB L2
// (DESIGN.md §5 "L2-resident pass 2 + join").
//
// Pass 2 splits each pass-1 partition into its 2^b2 co-partitions; every match of
// co-partition q lies in (R_q, S_q), so the join of q can start as soon as pass 2
// has finished q's pass-1 partition -- it does not need the whole pass. Two kernels (pass 2,
// then join) write 2w B/tuple to HBM and read them back; here:
//   * Roles per SM: the first fz_pass_slots blocks that start on an SM (per-SM slot counter on
//     %smid) run pass 2 (pass_body<FUSE>), the others run the join (join_body<FUSE>); pass-2
//     blocks join too once no pass-2 unit is left. Pass-2 units are claimed from a global
//     counter in pass-1-partition order, join items in co-partition order (the same order).
//   * Completion: each pass-2 warp signals its part of a unit (fence.acq_rel.gpu + red) on the
//     unit's pass-1 partition; a join item waits (ld.acquire.gpu) until its partition's count
//     is complete. Only pass-2 units wait on the join (throttle, bounded window of partitions in
//     flight), and never on a partition they still owe a signal, so the kernel cannot deadlock
//     whatever the block placement.
//   * L2 residency: pass 2 reads T1 evict-first and writes T2 with write-back stores; the join
//     reads T2 through L2 only and streams the pairs out evict-first, so HBM does not see the
//     2w B/tuple read-back of T2.
// Measured on B200 (c3): SLOWER than the separate kernels (fused kernel 1.8-2.2 ms vs pass 2 +
// join 1.6 ms). Both phases are latency/issue-bound (76 % / 65 % of HBM bandwidth as separate
// kernels), so splitting each SM between the roles halves each role's latency hiding while the
// saved HBM bytes were not the limit. Kept opt-in (HJ_OPT_FUSE) for that measurement. Also
// tried: discard.global.L2 of consumed co-partition lines -- slower (+0.7 ms) and it returned
// wrong results on repeated calls, so it was removed.
#pragma once
#include "hj_join.cuh"
#include "hj_partition.cuh"

namespace hj {

constexpr int FZ_NT = 512;          // block size: pass 2 uses all 512 threads,
constexpr int FZ_JOIN_NT = 480;     // the join 15 compute warps + 1 scheduler warp
constexpr int FZ_JOIN_SPT = 8;
static_assert(FZ_NT / 32 == FZ_PASS_WARPS, "pass-2 warps signal once per unit each");
static_assert(FZ_JOIN_NT / 32 == FZ_JOIN_WARPS, "join warps count once per item each");

template <typename K>
constexpr int fz_items() {
  return sizeof(K) == 4 ? 8 : 4;  // pass-2 unit = 512 x items tuples (32 KB)
}

template <typename K, bool MAT>
__global__ void __launch_bounds__(FZ_NT, 2) k_fused(Plan P) {
  __shared__ uint32_t s_role;
  // slot 0 of every SM always runs pass 2 (so some block does, whatever the placement)
  if (threadIdx.x == 0) s_role = atomicAdd(&P.fz[FZ_SLOT + (sm_id() & (FZ_NSLOT - 1))], 1u) < max(P.fz_pass_slots, 1u);
  __syncthreads();
  if (s_role) {
    pass_body<K, 2, FZ_NT, fz_items<K>(), false, false, true>(P, P.b2);
    __syncthreads();  // the join reuses the dynamic shared memory
  }
  join_body<K, FZ_JOIN_NT, FZ_JOIN_SPT, MAT, 1, false, true>(P);
}

}  // namespace hj
