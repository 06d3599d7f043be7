// hj_exchange.cuh -- kernels of the direct-store multi-GPU exchange (include/hj.h hj_xd_*,
// SURVEY.md §8(e)). The tuples themselves move inside pass 1 (k_pass<MODE 1>
// with the rank-widened digit): its reservation cursors are pre-set so every run lands at its
// final place in the owning rank's receive window, reached through a CUDA-IPC peer mapping
// (NVLink / NVSwitch stores on a multi-GPU node). What is left for this header is the count-row
// hand-off and the cross-rank barrier.
#pragma once

#include "hj_common.cuh"

namespace hj {

constexpr int XD_MAX = 64;  // HJ_XD_MAX_RANKS

// Board window (slot 2) of every rank, in uint64 words (include/hj.h HJ_XD_BOARD_BYTES):
constexpr int XB_FLAGS_B = 0;                 // [G] barrier flags (hj_xd_barrier; phase B of hj_xd_join)
constexpr int XB_FLAGS_A = 64;                // [G] phase A: source s published its totals
constexpr int XB_FLAGS_C = 128;               // [G] phase C: source s published its results
constexpr int XB_TOT = 192;                   // [src][2][dst] tuples of relation r src sends to dst
constexpr int XB_RES = XB_TOT + XD_MAX * 2 * XD_MAX;  // [src][2] (matches, checksum) of source s
constexpr int XB_WORDS = XB_RES + 2 * XD_MAX;

// this rank's per-destination count rows -> row `rank` of every destination's window header
struct XdRows {
  const uint32_t* cnt[2];  // [G][rowlen] q-order counts of R / S (the histogram's output)
  uint32_t* dst[2][XD_MAX];  // window header of rank j, already offset to row `rank`
  uint32_t rowlen;           // 2^local_bits
  const uint32_t* skip;      // hj_xd_join: non-zero = windows too small this call (write nothing)
};

// grid (G, 2, Z): blocks (j, r, *) copy relation r's row j to rank j, 16-byte stores when
// aligned, the row split over the Z blocks (a row is up to 2^20 words)
__global__ void __launch_bounds__(256) k_xd_rows(XdRows a) {
  if (a.skip && *a.skip) return;
  const int j = blockIdx.x, r = blockIdx.y;
  const uint32_t* src = a.cnt[r] + (size_t)j * a.rowlen;
  uint32_t* dst = a.dst[r][j];
  const uint32_t t0 = blockIdx.z * blockDim.x + threadIdx.x, step = gridDim.z * blockDim.x;
  const bool vec = (a.rowlen & 3) == 0 && ((reinterpret_cast<uintptr_t>(src) | reinterpret_cast<uintptr_t>(dst)) & 15) == 0;
  if (vec) {
    const uint4* s4 = reinterpret_cast<const uint4*>(src);
    uint4* d4 = reinterpret_cast<uint4*>(dst);
    for (uint32_t i = t0; i < a.rowlen / 4; i += step) d4[i] = s4[i];
  } else {
    for (uint32_t i = t0; i < a.rowlen; i += step) dst[i] = src[i];
  }
}

struct XdBarrier {
  unsigned long long* flags[XD_MAX];  // flag window of rank j (this process's mapping)
  const unsigned long long* own;      // this rank's flag window
  unsigned long long epoch;
  unsigned long long timeout_ns;
  uint32_t* err;  // mapped pinned host word: set to 1 on timeout
  int G, rank;
};

__device__ __forceinline__ void st_release_sys(unsigned long long* a, unsigned long long v) {
  asm volatile("st.release.sys.global.u64 [%0], %1;" ::"l"(a), "l"(v) : "memory");
}
__device__ __forceinline__ unsigned long long ld_acquire_sys(const unsigned long long* a) {
  unsigned long long v;
  asm volatile("ld.acquire.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(a) : "memory");
  return v;
}

// One block. Every thread first fences at system scope (the pass-1 peer stores of the previous
// kernel on this stream are complete at kernel boundaries; the fence orders them before the
// flag for any observer), thread j < G publishes the epoch to flag [rank] of rank j, then waits
// for flag [j] of its own window to reach the epoch. A %globaltimer deadline bounds every wait:
// a peer that never arrives costs timeout_ns, raises *err and never hangs the device.
__global__ void __launch_bounds__(XD_MAX) k_xd_barrier(XdBarrier b) {
  const int t = threadIdx.x;
  asm volatile("fence.sc.sys;" ::: "memory");
  __syncthreads();
  if (t < b.G) st_release_sys(b.flags[t] + b.rank, b.epoch);
  if (t < b.G) {
    const unsigned long long t0 = global_ns();
    while (ld_acquire_sys(b.own + t) < b.epoch) {
      if (global_ns() - t0 > b.timeout_ns) {  // site 2: the barrier (phase B); bit 4+: the missing rank
        asm volatile("st.relaxed.sys.global.u32 [%0], %1;" ::"l"(b.err), "r"(2u | ((uint32_t)t << 4)) : "memory");
        break;
      }
      __nanosleep(256);
    }
  }
  __syncthreads();
  asm volatile("fence.sc.sys;" ::: "memory");
}

// wait (acquire, system scope) until flags[t] >= epoch for every t < G; thread t waits on flag t
__device__ __forceinline__ void xd_wait_all(const unsigned long long* flags, int G, unsigned long long epoch,
                                            unsigned long long timeout_ns, uint32_t* err, uint32_t site) {
  const int t = threadIdx.x;
  if (t < G) {
    const unsigned long long t0 = global_ns();
    while (ld_acquire_sys(flags + t) < epoch) {
      if (global_ns() - t0 > timeout_ns) {  // site: 1 totals (phase A), 3 results (phase C); bit 4+: rank
        asm volatile("st.relaxed.sys.global.u32 [%0], %1;" ::"l"(err), "r"(site | ((uint32_t)t << 4)) : "memory");
        break;
      }
      __nanosleep(128);
    }
  }
  __syncthreads();
}

// ---- hj_xd_join: the whole exchange driven from the device (no host round trip) --------------
struct XdJoin {
  unsigned long long* board[XD_MAX];   // board window of rank j (this process's mapping)
  const unsigned long long* own;       // this rank's board
  const unsigned long long* pst[2];    // this rank's pass-1 piece starts (send plan), [2^(g+b1) + 1]
  unsigned long long* cur1[2];         // pass-1 cursors to set (send plan)
  uint32_t* rows0[2];                  // this rank's own window headers (zeroed on overflow)
  const unsigned long long* res;       // this rank's join results (matches, checksum)
  unsigned long long* sums;            // -> (matches, checksum) summed over ranks
  uint32_t* overflow;                  // -> 1 if some window is too small (all ranks agree)
  uint32_t* err;                       // mapped pinned host word: a wait timed out
  long long delta[2][XD_MAX];          // element offset of rank j's window tuples from this rank's
  long long scratch[2];                // ... and of the local scratch buffer (overflow)
  unsigned long long cap[2][XD_MAX];   // tuples every rank's window holds
  unsigned long long epoch, timeout_ns;
  uint32_t rows_words;                 // G * 2^local_bits
  int G, rank, b1;
};

// phase A: this rank's destination totals (from its pass-1 piece starts) -> tot[rank][r][*] of
// every rank's board, then flag A[rank] of every board (release after a system fence)
__global__ void __launch_bounds__(256) k_xd_totals(XdJoin a) {
  const int G = a.G;
  for (int i = threadIdx.x; i < G * 2 * G; i += blockDim.x) {
    const int j = i / (2 * G), r = (i / G) % 2, d = i % G;  // board of rank j, relation r, destination d
    const unsigned long long v = a.pst[r][(size_t)(d + 1) << a.b1] - a.pst[r][(size_t)d << a.b1];
    a.board[j][XB_TOT + ((size_t)a.rank * 2 + r) * XD_MAX + d] = v;
  }
  asm volatile("fence.sc.sys;" ::: "memory");
  __syncthreads();
  if (threadIdx.x < G) st_release_sys(a.board[threadIdx.x] + XB_FLAGS_A + a.rank, a.epoch);
}

// wait for every rank's totals, then set this rank's pass-1 cursors: digit D = (j, d1) starts at
// rank j's window, after the runs of sources s < rank for j (source-major), at d1's offset in
// this rank's run for j. If any rank's window is too small every rank sees it (same board):
// cursors go to the local scratch buffer, this rank's count-row headers are zeroed (its pass 2
// and join then do nothing) and the host grows the windows and calls again.
__global__ void __launch_bounds__(1024) k_xd_cursors(XdJoin a) {
  const int G = a.G;
  xd_wait_all(a.own + XB_FLAGS_A, G, a.epoch, a.timeout_ns, a.err, 1u);
  __shared__ unsigned long long s_seg[2][XD_MAX];
  __shared__ uint32_t s_over;
  if (threadIdx.x == 0) s_over = 0;
  __syncthreads();
  const unsigned long long* tot = a.own + XB_TOT;
  if (threadIdx.x < 2 * G) {
    const int r = threadIdx.x / G, j = threadIdx.x % G;
    unsigned long long seg = 0, all = 0;
    for (int s = 0; s < G; ++s) {
      const unsigned long long v = ld_acquire_sys(tot + ((size_t)s * 2 + r) * XD_MAX + j);
      if (s < a.rank) seg += v;
      all += v;
    }
    s_seg[r][j] = seg;
    if (all > a.cap[r][j]) atomicOr(&s_over, 1u);
  }
  __syncthreads();
  const bool over = s_over != 0;
  const uint32_t F1 = (uint32_t)G << a.b1;
  for (uint32_t i = threadIdx.x; i < 2 * F1; i += blockDim.x) {
    const int r = i >= F1;
    const uint32_t D = i - r * F1, j = D >> a.b1;
    const unsigned long long p = a.pst[r][D];
    a.cur1[r][D] = over ? (unsigned long long)a.scratch[r] + p
                        : (unsigned long long)a.delta[r][j] + s_seg[r][j] + (p - a.pst[r][(size_t)j << a.b1]);
  }
  if (over) {
    for (uint32_t i = threadIdx.x; i < a.rows_words; i += blockDim.x) a.rows0[0][i] = a.rows0[1][i] = 0;
    if (threadIdx.x == 0) *a.overflow = 1;
  }
}

// phase C: this rank's (matches, checksum) -> res[rank] of every board, flag C; wait for every
// rank's, sum them (mod 2^64) into a.sums
__global__ void __launch_bounds__(XD_MAX) k_xd_results(XdJoin a) {
  const int G = a.G, t = threadIdx.x;
  if (t < G) {
    a.board[t][XB_RES + 2 * a.rank] = a.res[0];
    a.board[t][XB_RES + 2 * a.rank + 1] = a.res[1];
  }
  asm volatile("fence.sc.sys;" ::: "memory");
  __syncthreads();
  if (t < G) st_release_sys(a.board[t] + XB_FLAGS_C + a.rank, a.epoch);
  xd_wait_all(a.own + XB_FLAGS_C, G, a.epoch, a.timeout_ns, a.err, 3u);
  if (t == 0) {
    unsigned long long m = 0, c = 0;
    for (int s = 0; s < G; ++s) {
      m += ld_acquire_sys(a.own + XB_RES + 2 * s);
      c += ld_acquire_sys(a.own + XB_RES + 2 * s + 1);
    }
    a.sums[0] = m;
    a.sums[1] = c;
  }
}

}  // namespace hj
