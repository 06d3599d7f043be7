// hj_api.cu -- the C-ABI of include/hj.h: context, workspace, planning of launch shapes and
// the launch sequence of one join. Single translation unit (kernels in the .cuh headers).
#include <cuda_runtime.h>

#include <algorithm>
#include <cmath>
#include <cstdarg>
#include <cstdio>
#include <cstring>
#include <map>
#include <string>
#include <tuple>
#include <vector>

#include "../../include/hj.h"
#include "hj_exchange.cuh"
#include "hj_join.cuh"
#include "hj_partition.cuh"
#include "hj_pass_ws.cuh"
#include "hj_variants.cuh"

using namespace hj;

#define HJ_STR2(x) #x
#define HJ_STR(x) HJ_STR2(x)

namespace {

thread_local std::string g_create_error;

// Join kernel shapes selectable with HJ_OPT_JOIN_VARIANT (tuning; results never change).
//   variant: compute threads, S tuples / thread / round, min blocks / SM, R tile buffers
struct JoinShape {
  int nt, spt, minb, rbuf, nbsh;  // nbsh: hash slots = 2^(ceil(log2 C_R) - nbsh)
  bool h16;                       // 16-bit chain heads
  bool pf;                        // next probe round's S loads issued before the current walk
  bool l2pf;                      // claimed item's R chunk + first S round prefetched into L2
  int spf = 0;                    // S stream prefetched into L2 this many probe rounds ahead (0 = off)
  bool bf = true;                 // branch-free first chain step for every tuple of a round
};
// 0-2 are the defaults (join_variant below); 3-5 are kept as measured alternatives (round 1 swept
// 46 shapes; the slower ones were removed)
constexpr JoinShape JOIN_SHAPES[] = {
    {256, 6, 3, 1, 1, false, true, true},      // 0: 4 B count
    {256, 8, 3, 1, 1, false, false, true, 2},  // 1: 4 B materialize
    {512, 1, 2, 1, 1, false, true, true, 0, false},  // 2: 8 B (both modes), round-1 shape
    {256, 8, 3, 1, 1},                         // 3: no prefetching
    {256, 8, 2, 2, 1},                         // 4: double-buffered R tile
    {224, 8, 4, 1, 1, true},                   // 5: 16-bit heads, 4 blocks / SM
    {512, 2, 2, 1, 1, false, true, true, 0, false},  // 6: 8 B, two tuples per thread (c5_gpu join 2.71 vs 2.45 ms)
    {512, 2, 2, 1, 1, false, true, true},             // 7: 8 B, branch-free first step (2.60 ms; 256 x 4: 3.23)
    {512, 1, 2, 1, 0, false, true, true, 0, false},  // 8: 8 B default: shape 2 with twice the hash slots
};
constexpr int JOIN_NVARIANTS = sizeof(JOIN_SHAPES) / sizeof(JOIN_SHAPES[0]);
constexpr int HIST_NT = 1024;

struct DevBuf {
  void* p = nullptr;
  size_t bytes = 0;
  bool ws = false;  // carved from the caller's workspace (hj_set_workspace), not ctx-owned
};

struct HostPlan;

// hj_join_async: a call whose result readback is enqueued but not yet waited for. Each slot owns
// its events and pinned result words, so calls can be queued back to back on the stream.
constexpr int MAX_PENDING = HJ_MAX_PENDING;
struct Pending {
  hj_result* res = nullptr;
  cudaEvent_t ev[7] = {};
  unsigned long long* h = nullptr;  // pinned: results readback of this call
  int B = 0;
  bool mat = false, bc = false, recv = false, timing = false;
  unsigned long long out_cap = 0;
  const void* out_r = nullptr;
  const void* out_s = nullptr;
  uint32_t launches = 0;
};

struct Ctx {
  int device = 0;
  int key_bytes = 4, pay_bytes = 4;
  cudaStream_t stream = nullptr;
  cudaStream_t own_stream = nullptr;
  cudaStream_t h2d_stream = nullptr, d2h_stream = nullptr;  // streaming hj_join_host (NEXT-3)
  cudaEvent_t sev[12] = {};                                  // streaming events
  DevBuf sin[2][2];                                          // S chunk double buffers [buf][keys/pays]
  void* h_cur = nullptr;                                     // pinned: output cursor per chunk
  int num_sms = 148;
  size_t smem_optin = 0;
  std::string err;
  // options
  int64_t opt_cap_r = 0, opt_chunk_s = 0, opt_out_cap = 0, opt_timing = 1, opt_bps = 0, opt_join_variant = -1,
          opt_pass_nt = 0, opt_stream_chunk = 0, opt_join_algo = 0, opt_graph = 0, opt_pass_l2pf = 2, opt_pass1_bits = 0,
          opt_partitioner = 0, opt_pass_variant = 0, opt_mat_chk = 1, opt_pass_ws = 1, opt_pdl = 0;
  DevBuf bc_pool1[2], bc_pool2[2], bc_meta;  // HJ_OPT_PARTITIONER = 1 (NEXT-1 bucket chains)
  // workspace
  DevBuf t1[2], t2[2], meta, out_r, out_s, in[4], xsend[2], xcnt[2], np_heads, np_next;
  void* h_res = nullptr;  // pinned host: results readback
  void* h_out = nullptr;  // pinned host: materialized pairs (hj_join_host)
  size_t h_out_bytes = 0;
  DevBuf part_off_host_dummy;
  cudaEvent_t ev[8] = {};
  uint32_t launches = 0;
  std::map<std::tuple<const void*, int, size_t>, int> occ;  // occupancy() cache
  // HJ_OPT_GRAPH: the launch sequence of the last hj_join, captured once and replayed while the
  // call signature (columns, sizes, radix bits, mode, workspace) is unchanged
  // direct-store exchange (hj_xd_*): windows [R recv, S recv, flags], the plan of the last
  // hj_xd_count, its pass-1 piece starts, the barrier epoch and the timeout word
  DevBuf xd_win[3], xd_meta;
  HostPlan* xd_hp = nullptr;
  Plan* xd_P = nullptr;
  std::vector<unsigned long long> xd_pst[2];
  unsigned long long* h_xd_cur = nullptr;  // pinned: cursor table upload / totals board readback (64 KB)
  uint32_t* h_xd_err = nullptr;            // pinned, mapped: barrier timeout flag
  uint32_t* d_xd_err = nullptr;
  unsigned long long xd_epoch = 0;
  // caller-provided workspace (hj_set_workspace): hj_join carves every device buffer it needs
  // from [ws, ws + ws_bytes) in a fixed order (bump pointer reset per call) instead of allocating;
  // `dry` = hj_workspace_bytes: the allocation steps only sum the sizes
  char* ws = nullptr;
  size_t ws_bytes = 0, ws_off = 0;
  bool use_ws = false;  // inside hj_join with a workspace set
  std::vector<DevBuf*> ws_bufs;
  bool dry = false;
  size_t dry_bytes = 0;
  cudaGraphExec_t graph = nullptr;
  unsigned long long graph_key[16] = {};
  bool capturing = false;  // a graph capture is in progress on c->stream
  uint32_t graph_launches = 0;
  // hj_join_async: ring of pending calls (issue order from pend_head); `async` = the slot the
  // call being enqueued fills (finish_join then enqueues its readback and returns)
  Pending pend[MAX_PENDING];
  int pend_head = 0, pend_n = 0;
  Pending* async = nullptr;
  cudaEvent_t ev_own[7] = {};  // the ctx's own timing events (c->ev[0..6] outside async calls)
};

int fail(Ctx* c, int code, const char* fmt, ...) {
  char buf[512];
  va_list ap;
  va_start(ap, fmt);
  vsnprintf(buf, sizeof buf, fmt, ap);
  va_end(ap);
  if (c) c->err = buf;
  else g_create_error = buf;
  return code;
}

#define CUDA_TRY(c, expr)                                                                         \
  do {                                                                                            \
    cudaError_t e_ = (expr);                                                                      \
    if (e_ != cudaSuccess)                                                                        \
      return fail((c), e_ == cudaErrorMemoryAllocation ? HJ_ERR_OOM : HJ_ERR_CUDA, "%s: %s (%s:%d)", \
                  #expr, cudaGetErrorString(e_), __FILE__, __LINE__);                             \
  } while (0)

size_t align_up(size_t x, size_t a) { return (x + a - 1) / a * a; }

void drop_graph(Ctx* c) {
  if (c->graph) cudaGraphExecDestroy(c->graph);
  c->graph = nullptr;
}

// Device buffer of at least `bytes` for this call. Three modes:
//   dry (hj_workspace_bytes): only sum the 256-byte aligned sizes;
//   workspace (hj_join after hj_set_workspace): carve from the caller's buffer, never allocate;
//   otherwise a ctx-owned cudaMalloc, kept and reused while large enough.
// No buffer is zeroed here: every call zeroes exactly what it reads before writing (the
// planner's counters / results region, the bucket-chain states) with cudaMemsetAsync.
int ensure(Ctx* c, DevBuf& b, size_t bytes) {
  if (c->dry) {
    c->dry_bytes += align_up(bytes, 256);
    return HJ_OK;
  }
  if (c->use_ws) {
    if (b.ws && b.p && b.bytes >= bytes) return HJ_OK;  // carved earlier in this call
    if (b.p && !b.ws) {  // a ctx-owned buffer from a call without workspace
      cudaStreamSynchronize(c->stream);
      cudaFree(b.p);
    }
    const size_t need = align_up(bytes, 256);
    if (c->ws_off + need > c->ws_bytes)
      return fail(c, HJ_ERR_WORKSPACE, "workspace of %zu bytes too small (needs > %zu; see hj_workspace_bytes)",
                  c->ws_bytes, c->ws_off + need);
    b.p = c->ws + c->ws_off;
    b.bytes = bytes;
    b.ws = true;
    c->ws_off += need;
    c->ws_bufs.push_back(&b);
    return HJ_OK;
  }
  if (b.bytes >= bytes && b.p && !b.ws) return HJ_OK;
  if (b.p && !b.ws) {  // earlier work of this ctx may still read it (e.g. an asynchronous pass 1)
    cudaStreamSynchronize(c->stream);
    cudaFree(b.p);
  }
  b.p = nullptr;
  b.bytes = 0;
  b.ws = false;
  drop_graph(c);  // a captured launch sequence may hold the old address
  if (bytes == 0) return HJ_OK;
  CUDA_TRY(c, cudaMalloc(&b.p, bytes));
  b.bytes = bytes;
  return HJ_OK;
}

// start of an hj_join call with a workspace: buffers are carved again from offset 0 (same sizes
// and order -> same addresses, so a captured graph stays valid)
void ws_begin(Ctx* c) {
  for (DevBuf* b : c->ws_bufs)
    if (b->ws) {  // (a buffer another entry point re-allocated since is ctx-owned now)
      b->p = nullptr;
      b->bytes = 0;
      b->ws = false;
    }
  c->ws_bufs.clear();
  c->ws_off = 0;
}

// does the materialized output need (re)allocation for `pairs` pairs?
bool out_short(const Ctx* c, unsigned long long pairs) {
  return c->dry || c->out_r.bytes < pairs * c->pay_bytes || c->out_s.bytes < pairs * c->pay_bytes;
}

int ilog2_ceil(unsigned long long x) {
  int l = 0;
  while ((1ull << l) < x) ++l;
  return l;
}

// Host-side plan of one call: radix bits, capacities, launch shapes, metadata layout.
struct HostPlan {
  int B = 0, b1 = 0, b2 = 0, gsh = 0;
  int g = 0, nsrc = 1, mode = PLAN_FULL;
  uint32_t CR = 0, CS = 0, C2 = 0;
  int lg_nb = 6;
  size_t join_smem = 0;
  int tile = 0;
  // metadata offsets (bytes) inside ctx->meta
  size_t o_cnt[2], o_off[2], o_cur1[2], o_cur2[2], o_pst[2], o_cst[2], o_hot[2], o_ist, o_ist2, o_counters, o_results;
  size_t zero_bytes = 0;  // [0, zero_bytes) is memset to 0 per call
  size_t meta_bytes = 0;
  int pb() const { return g + b1; }
  int qbits() const { return g + B; }
  uint32_t npieces() const { return (uint32_t)nsrc << pb(); }
};

template <typename K>
constexpr int pass_items() {
  return sizeof(K) == 4 ? 8 : 4;  // 8192-tuple tiles of 8 B, 4096-tuple tiles of 16 B (64 KB)
}

// default join shape per key width and output mode (measured with tools/tune.py on B200):
//   4 B materialize -> shape 1 (256 x 8, L2 prefetch of the next item and of the S stream 2
//                      rounds ahead: c3 join 0.749 -> 0.704 ms before the 32-bit-shared-address
//                      probe, 0.646 after)
//   4 B count       -> shape 0 (256 x 6, next round's S in registers + L2 prefetch of the next
//                      item: c2 0.873 -> 0.814 ms; streaming S through L2 was slower here)
//   8 B             -> shape 8 (512 x 1, two blocks per SM: the 16-byte R tile limits blocks to
//                      two per SM, so more threads per block -- not more tuples per thread --
//                      hide the chain-walk latency: c5_gpu join 3.54 -> 2.69 ms in round 1; 512 x 2:
//                      2.90, 640 x 1: 2.85, 768 x 1: 3.34) with twice the hash slots: fmix64 keys hash
//                      to random slots, so chains at load factor 1 average 1.5 entries per hit (2.45
//                      -> 2.16 ms; 16-bit heads with 2x / 4x slots 2.56 / 2.82, branch-free first
//                      step 2.30-2.40; 4-byte dense keys hash without collisions: c2 2x slots 0.58 -> 0.63)
int join_variant(const Ctx* c, bool mat) {
  if (c->opt_join_variant >= 0) return (int)c->opt_join_variant;
  if (c->key_bytes == 8) return 8;
  return mat ? 1 : 0;
}

int pass_threads(const Ctx* c, int fanout_bits, int items) {
  if (c->opt_pass_nt) return (int)c->opt_pass_nt == 512 && (1 << fanout_bits) <= 512 ? 512 : 1024;
  return (512 * items) >> fanout_bits >= 32 ? 512 : 1024;
}

// the warp-specialized pass (hj_pass_ws.cuh) for a fan-out of 2^bits: fan-out <= WS_MAXF
// (shared-memory budget); its unit is a 60 KB tile. The bucket-chain partitioner has it for the
// default role split only.
bool use_ws(const Ctx* c, int bits) {
  return c->opt_pass_ws && (1 << bits) <= WS_MAXF && (c->opt_partitioner == 0 || c->opt_pass_ws == 1);
}
// role split: HJ_OPT_PASS_WS = 1 (default: 20 compute warps; measured on B200, c3 pass 1 / pass 2:
// 16 warps x 16 tuples 1.01 / 0.97 ms (spills), 18: 0.82 / 0.87, 20: 0.80 / 0.82, 21: 0.81 / 0.83,
// 22: 0.84 / 0.85, 24 x 8 tuples: 0.93 / 0.93; the lock-step k_pass: 0.94 / 0.85) or an explicit
// number of compute warps among WS_CWS
#define WS_CWS(X) X(18) X(20) X(22)
// (8-byte tuples move twice the bytes per tuple through the writer warps: 18 compute warps + 13
// writers measured faster, c5_gpu 8.42 -> 8.20 ms per call; the bucket-chain kernels are built
// for 20)
int ws_cw(const Ctx* c) {
  if (c->opt_pass_ws != 1) return (int)c->opt_pass_ws;
  return c->key_bytes == 8 && c->opt_partitioner == 0 ? 18 : 20;
}
uint32_t ws_tile(const Ctx* c) {
  const int cw = ws_cw(c);
#define WS_TILE_CASE(N) \
  if (cw == N) return c->key_bytes == 4 ? WsShape<uint32_t, N>::TILE : WsShape<uint64_t, N>::TILE;
  WS_CWS(WS_TILE_CASE)
#undef WS_TILE_CASE
  return 0;
}

int choose_bits(unsigned long long nR) {
  // mean R co-partition ~4096 tuples: the paper's shared-memory reservation
  if (nR <= 4096) return 0;
  int B = ilog2_ceil((nR + 4095) / 4096);
  return std::min(B, 20);
}

// pass-1 bits of the exchange: pass 1's fan-out (rank bits + b1) and the
// receiver's pieces (sources x 2^b1) stay <= 2^10, so b1 = min(ceil(B/2), 10 - log2 G); sender
// and receiver derive the same b1 (c5 at G = 8: B = 16 -> 7 + 9)
int xchg_b1(int G, int B) {
  const int gl = ilog2_ceil((unsigned long long)std::max(G, 1));
  int b1 = (B + 1) / 2;
  if (gl > 0 && b1 > 10 - gl) b1 = std::max(0, 10 - gl);
  return b1;
}

// mode PLAN_FULL: one GPU; PLAN_SEND: exchange sender (g rank bits); PLAN_RECV: exchange
// receiver (nsrc sources). nR / nS are the tuples this GPU partitions / joins.
// nR_est: the R tuples the join capacities are sized for (0 = nR). The exchange receiver's buffers
// are sized by its window capacity, its join by the rows it expects (its share).
int make_plan(Ctx* c, HostPlan& hp, unsigned long long nR, unsigned long long nS, int radix_bits, bool mat, int g = 0,
              int nsrc = 1, int mode = PLAN_FULL, unsigned long long nR_est = 0) {
  const size_t tb = (size_t)c->key_bytes + c->pay_bytes;  // AoS tuple bytes
  hp.B = radix_bits < 0 ? choose_bits(nR) : radix_bits;
  if (hp.B > 20) return fail(c, HJ_ERR_UNSUPPORTED, "radix_bits %d > 20", hp.B);
  hp.b1 = (hp.B + 1) / 2;  // reading S6; HJ_OPT_PASS1_BITS overrides on one GPU (results never change)
  const bool xchg = mode != PLAN_FULL || g > 0 || nsrc > 1;
  if (xchg) hp.b1 = xchg_b1(std::max(1 << g, nsrc), hp.B);
  else if (c->opt_pass1_bits > 0 && hp.B >= 2) hp.b1 = (int)std::min<int64_t>(c->opt_pass1_bits, hp.B - 1);
  hp.b2 = hp.B - hp.b1;
  hp.gsh = hp.B;
  if (mode == PLAN_SEND) {  // the sender counts and lays out only its (rank, d1) pieces
    hp.B = hp.b1;
    hp.b2 = 0;
  }
  hp.g = g;
  hp.nsrc = nsrc;
  hp.mode = mode;
  if (hp.pb() > 10 || hp.b2 > 10 || hp.npieces() > 1024)
    return fail(c, HJ_ERR_UNSUPPORTED, "pass fan-out too large (g=%d b1=%d b2=%d sources=%d)", g, hp.b1, hp.b2, nsrc);
  const int items = c->key_bytes == 4 ? pass_items<uint32_t>() : pass_items<uint64_t>();
  // pass tiles: two 512-thread blocks per SM when a 512-thread tile still averages >= 32 tuples
  // per digit run (measured: shorter runs cost more than the extra block's overlap), else one
  // 1024-thread block. The pass-2 chunk is that kernel's tile.
  hp.tile = use_ws(c, hp.pb()) ? ws_tile(c) : pass_threads(c, hp.pb(), items) * items;
  hp.C2 = use_ws(c, hp.b2) ? ws_tile(c) : (uint32_t)(pass_threads(c, hp.b2, items) * items);

  // join capacities
  const unsigned long long mean = ((nR_est ? std::min(nR_est, nR) : nR) + (1ull << hp.B) - 1) >> hp.B;
  size_t cap_max_smem = c->smem_optin ? c->smem_optin : 227 * 1024;
  uint32_t CR;
  if (c->opt_cap_r > 0) CR = (uint32_t)std::min<int64_t>(c->opt_cap_r, 65534);
  else CR = (uint32_t)std::min<unsigned long long>(align_up(mean + 5 * (unsigned long long)sqrt((double)mean) + 64, 128), 16384);
  CR = std::max<uint32_t>(CR, c->opt_cap_r > 0 ? 1 : 512);
  uint32_t CS;
  if (c->opt_chunk_s > 0) CS = (uint32_t)std::min<int64_t>(c->opt_chunk_s, 1ll << 30);
  else CS = std::max<uint32_t>(8 * CR, 32768);
  const JoinShape& JS = JOIN_SHAPES[join_variant(c, mat)];
  const int rbuf = JS.rbuf, nbsh = JS.nbsh;
  const size_t head_bytes = JS.h16 ? 2 : 4;
  int lg_nb = std::max(6, ilog2_ceil(CR) - nbsh);
  auto join_smem = [&](uint32_t cr, int lg) {  // R tile buffer(s) (TMA) + heads + next
    return (size_t)rbuf * ((cr + 3) & ~1u) * tb + (head_bytes << lg) + (size_t)(cr + 1) * 2;
  };
  const size_t join_cap = cap_max_smem - 8 * 1024;
  while (join_smem(CR, lg_nb) > join_cap && CR > 256) {
    CR /= 2;
    lg_nb = std::max(6, ilog2_ceil(CR) - nbsh);
  }
  hp.CR = CR;
  hp.CS = CS;
  hp.lg_nb = lg_nb;
  hp.join_smem = join_smem(CR, lg_nb);

  // metadata layout
  const size_t nq = (size_t)1 << hp.qbits(), F1 = (size_t)1 << hp.pb(), npc = hp.npieces();
  size_t o = 0;
  auto take = [&](size_t bytes) {
    size_t r = o;
    o = align_up(o + bytes, 256);
    return r;
  };
  // zeroed region first
  hp.o_counters = take(64);
  hp.o_results = take(64);
  for (int r = 0; r < 2; ++r) hp.o_cnt[r] = take(nq * 4);  // (the receiver's own histogram too)
  hp.zero_bytes = o;
  for (int r = 0; r < 2; ++r) {
    hp.o_off[r] = take((nq + 1) * 8);
    hp.o_cur1[r] = take(F1 * 8);
    hp.o_cur2[r] = take(nq * 8);
    hp.o_pst[r] = take((npc + 1) * 8);
    hp.o_cst[r] = take((npc + 1) * 4);
    hp.o_hot[r] = take((F1 + 1) * 4);
  }
  hp.o_ist = take((((size_t)1 << hp.B) + 1) * 4);
  hp.o_ist2 = take((((size_t)1 << hp.B) + 1) * 4);
  hp.meta_bytes = o;
  (void)nS;
  return HJ_OK;
}

template <typename K, int V, typename F>
void attr_join(F&& attr) {
  constexpr JoinShape S = JOIN_SHAPES[V];
  attr((const void*)k_join<K, S.nt, S.spt, false, S.minb, S.rbuf, S.h16, S.pf, S.l2pf, S.spf, true, S.bf>);
  attr((const void*)k_join<K, S.nt, S.spt, true, S.minb, S.rbuf, S.h16, S.pf, S.l2pf, S.spf, true, S.bf>);
  if constexpr (sizeof(K) == 4) {
    attr((const void*)k_join<K, S.nt, S.spt, false, S.minb, S.rbuf, S.h16, S.pf, S.l2pf, S.spf, false, S.bf>);
    attr((const void*)k_join<K, S.nt, S.spt, true, S.minb, S.rbuf, S.h16, S.pf, S.l2pf, S.spf, false, S.bf>);
  }
}

template <typename K, typename F>
void for_ws_variants(F&& attr) {
#define WS_ATTR_CASE(N)                                 \
  attr((const void*)k_pass_ws<K, 1, false, N>);        \
  attr((const void*)k_pass_ws<K, 1, true, N>);         \
  attr((const void*)k_pass_ws<K, 2, false, N>);
  WS_CWS(WS_ATTR_CASE)
#undef WS_ATTR_CASE
  attr((const void*)k_pass_ws<K, 1, false, 20, true>);
  attr((const void*)k_pass_ws<K, 2, false, 20, true>);
}

template <typename K>
int set_kernel_attrs(Ctx* c) {
  int rc = 0;
  auto attr = [&](const void* f) {
    cudaFuncAttributes fa;
    if (cudaFuncGetAttributes(&fa, f) != cudaSuccess ||
        cudaFuncSetAttribute(f, cudaFuncAttributeMaxDynamicSharedMemorySize,
                             (int)(c->smem_optin - fa.sharedSizeBytes)) != cudaSuccess)
      rc = -1;
  };
  // kernels without a shared-memory attribute are still touched here: under lazy module
  // loading (the CUDA 12 default) a kernel's first launch loads it, which can synchronize the
  // context -- inside hj_xd_join that would wait on kernels that wait on this rank
  auto load = [&](const void* f) {
    cudaFuncAttributes fa;
    if (cudaFuncGetAttributes(&fa, f) != cudaSuccess) rc = -1;
  };
  load((const void*)k_hist<K, false, false>);
  load((const void*)k_hist<K, false, true>);
  load((const void*)k_plan<false, true>);
  load((const void*)k_plan<false, false>);
  load((const void*)k_plan<true, true>);
  load((const void*)k_xd_rows);
  load((const void*)k_xd_totals);
  load((const void*)k_xd_cursors);
  load((const void*)k_xd_barrier);
  load((const void*)k_xd_results);
  attr((const void*)k_join_nlj<K, 256, false>);
  attr((const void*)k_join_nlj<K, 256, true>);
  attr((const void*)k_hist<K, true, false, true>);
  attr((const void*)k_hist<K, true, true, true>);
  attr((const void*)k_hist<K, true, false, false>);
  attr((const void*)k_hist<K, true, true, false>);
  load((const void*)k_hist_recv<K, false, false>);
  attr((const void*)k_hist_recv<K, true, true>);
  attr((const void*)k_hist_recv<K, true, false>);
  for_ws_variants<K>(attr);
  attr((const void*)k_pass<K, 1, 1024, pass_items<K>(), false>);
  attr((const void*)k_pass<K, 1, 1024, pass_items<K>(), true>);
  attr((const void*)k_pass<K, 2, 1024, pass_items<K>(), false>);
  attr((const void*)k_pass<K, 1, 512, pass_items<K>(), false>);
  attr((const void*)k_pass<K, 1, 512, pass_items<K>(), true>);
  attr((const void*)k_pass<K, 2, 512, pass_items<K>(), false>);
  attr((const void*)k_pass<K, 1, 1024, pass_items<K>(), false, true>);
  attr((const void*)k_pass<K, 1, 512, pass_items<K>(), false, true>);
  attr((const void*)k_pass<K, 2, 1024, pass_items<K>(), false, true>);
  attr((const void*)k_pass<K, 2, 512, pass_items<K>(), false, true>);
  attr((const void*)k_pass<K, 1, 512, 2 * pass_items<K>(), false, false, false>);
  attr((const void*)k_pass<K, 1, 512, 2 * pass_items<K>(), true, false, false>);
  attr((const void*)k_pass<K, 2, 512, 2 * pass_items<K>(), false, false, false>);
  attr((const void*)k_pass<K, 1, 512, 2 * pass_items<K>(), false, true, false>);
  attr((const void*)k_pass<K, 2, 512, 2 * pass_items<K>(), false, true, false>);
  attr_join<K, 0>(attr);
  attr_join<K, 1>(attr);
  attr_join<K, 2>(attr);
  attr_join<K, 3>(attr);
  attr_join<K, 4>(attr);
  attr_join<K, 5>(attr);
  attr_join<K, 6>(attr);
  attr_join<K, 7>(attr);
  attr_join<K, 8>(attr);
  return rc;
}

// resident blocks per SM of (kernel, block size, dynamic smem), cached per context: the occupancy
// query is host work on every launch otherwise (it sits between back-to-back calls)
int occupancy(Ctx* c, const void* f, int nt, size_t smem) {
  const auto key = std::make_tuple(f, nt, smem);
  auto it = c->occ.find(key);
  if (it != c->occ.end()) return it->second;
  int per_sm = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, f, nt, smem) != cudaSuccess) {
    cudaGetLastError();
    per_sm = 0;
  }
  c->occ[key] = per_sm;
  return per_sm;
}

int grid_for(Ctx* c, const void* f, int nt, size_t smem, unsigned long long units) {
  int per_sm = occupancy(c, f, nt, smem);
  if (per_sm < 1) per_sm = 1;
  if (c->opt_bps > 0) per_sm = std::min<int>(per_sm, (int)c->opt_bps);
  unsigned long long g = (unsigned long long)per_sm * c->num_sms;
  if (units < g) g = units;
  return (int)std::max<unsigned long long>(g, 1);
}

// Fill the device Plan for one call; rel 1 may be empty (hj_partition, hj_exchange_pack).
Plan device_plan(Ctx* c, const HostPlan& hp, const void* Rk, const void* Rp, unsigned long long nR, const void* Sk,
                 const void* Sp, unsigned long long nS, void* meta = nullptr) {
  Plan P;
  memset(&P, 0, sizeof P);
  char* m = (char*)(meta ? meta : c->meta.p);
  const void* ks[2] = {Rk, Sk};
  const void* ps[2] = {Rp, Sp};
  const unsigned long long ns[2] = {nR, nS};
  for (int r = 0; r < 2; ++r) {
    RelDev& d = P.rel[r];
    d.keys = ks[r];
    d.pays = ps[r];
    d.n = ns[r];
    d.t1 = c->t1[r].p;
    d.t2 = c->t2[r].p;
    d.cnt = (uint32_t*)(m + hp.o_cnt[r]);
    d.off = (unsigned long long*)(m + hp.o_off[r]);
    d.cur1 = (unsigned long long*)(m + hp.o_cur1[r]);
    d.cur2 = (unsigned long long*)(m + hp.o_cur2[r]);
    d.pst = (unsigned long long*)(m + hp.o_pst[r]);
    d.cst = (uint32_t*)(m + hp.o_cst[r]);
    d.hot = (uint32_t*)(m + hp.o_hot[r]);
    P.tiles1[r] = (ns[r] + hp.tile - 1) / hp.tile;
  }
  P.B = hp.B;
  P.b1 = hp.b1;
  P.b2 = hp.b2;
  P.g = hp.g;
  P.gsh = hp.gsh;
  P.nsrc = hp.nsrc;
  P.mode = hp.mode;
  P.C2 = hp.C2;
  P.tuple_bytes = c->key_bytes + c->pay_bytes;
  // measured (tools/tune.py pass_l2pf): 8 B tuples pass 1 4.02 -> 3.59 ms on c5_gpu; 4 B pass 1
  // slower (c3 0.939 -> 0.983), pass 2 unchanged -> auto (2) = on for 8-byte keys only
  P.pass_l2pf = c->opt_pass_l2pf == 2 ? (c->key_bytes == 8) : (c->opt_pass_l2pf ? 1 : 0);
  P.CR = hp.CR;
  P.lgCRp = 0;
  while ((2u << P.lgCRp) <= hp.CR) ++P.lgCRp;
  P.CS = hp.CS;
  P.ist = (uint32_t*)(m + hp.o_ist);
  P.ist2 = (uint32_t*)(m + hp.o_ist2);
  P.counters = (uint32_t*)(m + hp.o_counters);
  P.results = (unsigned long long*)(m + hp.o_results);
  P.mat_chk = c->opt_mat_chk ? 1 : 0;
  P.out_r = c->out_r.p;
  P.out_s = c->out_s.p;
  P.out_cap = std::min(c->out_r.bytes, c->out_s.bytes) / c->pay_bytes;
  P.H.B = hp.B;
  P.H.lg = hp.lg_nb;
  P.one = 1;
  {
    const int rem = 8 * c->key_bytes - hp.B;  // key bits above the radix field (64-bit keys fold to 32 first)
    const int bits = std::min(rem, 32);
    P.H.nfold = std::min(3, std::max(0, (bits + hp.lg_nb - 1) / hp.lg_nb - 1));
  }
  return P;
}

// launch on the ctx stream; HJ_OPT_PDL = 1: with programmatic stream serialization, so the
// kernel (which starts with pdl_wait) is scheduled while its predecessor's last blocks run
template <typename... KArgs, typename... Args>
cudaError_t launch_k(Ctx* c, void (*f)(KArgs...), dim3 grid, dim3 block, size_t smem, Args... args) {
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = grid;
  cfg.blockDim = block;
  cfg.dynamicSmemBytes = smem;
  cfg.stream = c->stream;
  cudaLaunchAttribute at[1];
  at[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
  at[0].val.programmaticStreamSerializationAllowed = 1;
  cfg.attrs = at;
  cfg.numAttrs = c->opt_pdl ? 1 : 0;
  return cudaLaunchKernelEx(&cfg, f, args...);
}

void mark(Ctx* c, int i) {
  // inside a graph capture the record must be an external event-record node to be timed
  if (c->opt_timing)
    cudaEventRecordWithFlags(c->ev[i], c->stream, c->capturing ? cudaEventRecordExternal : cudaEventRecordDefault);
}

// a1 (histogram), a2/a5 (planner), a3 (pass 1). PLAN_RECV skips a1 and a3 (counts and the
// pass-1 layout arrive through the exchange). Events 0..3.
template <typename K, int MODE, int NT, bool GD, bool BC = false>
int launch_pass(Ctx* c, const HostPlan& hp, const Plan& P, int fanout_bits);

// a2: the planner instance for this plan (several sources / join items)
int launch_plan(Ctx* c, const HostPlan& hp, const Plan& P) {
  const unsigned g = (unsigned)((((size_t)1 << hp.qbits()) + 1023) / 1024);
  const bool ms = P.nsrc > 1, it = P.mode != PLAN_SEND;
  cudaStream_t st = c->stream;
  if (ms) CUDA_TRY(c, launch_k(c, k_plan<true, true>, g, 1024, 0, P));
  else if (it) CUDA_TRY(c, launch_k(c, k_plan<false, true>, g, 1024, 0, P));
  else CUDA_TRY(c, launch_k(c, k_plan<false, false>, g, 1024, 0, P));
  CUDA_TRY(c, cudaGetLastError());
  c->launches += 1;
  return HJ_OK;
}

// a1 on the exchange receiver: its own histogram of what it received (k_hist_recv)
template <typename K>
int launch_hist_recv(Ctx* c, const HostPlan& hp, const Plan& P) {
  cudaStream_t st = c->stream;
  const bool smem = hp.B <= 16, c32 = hp.B <= 15;
  const size_t sm = smem ? (c32 ? ((size_t)4 << hp.B) : ((size_t)2 << hp.B)) : 0;
  const unsigned long long nR = P.rel[0].n, nS = P.rel[1].n;
  const void* f = !smem ? (const void*)k_hist_recv<K, false, false>
                        : c32 ? (const void*)k_hist_recv<K, true, true> : (const void*)k_hist_recv<K, true, false>;
  const int g = std::max(2, grid_for(c, f, HIST_NT, sm, (nR + nS + 4095) / 4096 + 2));
  uint32_t gr = (uint32_t)((double)g * (double)nR / (double)std::max<unsigned long long>(nR + nS, 1) + 0.5);
  gr = std::min<uint32_t>(std::max<uint32_t>(gr, 1), (uint32_t)g - 1);
  if (!smem) k_hist_recv<K, false, false><<<g, HIST_NT, 0, st>>>(P, gr);
  else if (c32) k_hist_recv<K, true, true><<<g, HIST_NT, sm, st>>>(P, gr);
  else k_hist_recv<K, true, false><<<g, HIST_NT, sm, st>>>(P, gr);
  CUDA_TRY(c, cudaGetLastError());
  c->launches += 1;
  return HJ_OK;
}

// stage: 0 = all of a1-a3; 1 = a1-a2 only (hj_xd_count); 2 = a3 only (hj_xd_store, after stage 1
// with the same plan)
template <typename K>
int launch_front(Ctx* c, const HostPlan& hp, const Plan& P, bool chunk = false, int stage = 0) {
  cudaStream_t st = c->stream;
  const bool gd = hp.g > 0;
  if (stage == 2) {
    mark(c, 2);
    int rc = hp.tile == 512 * pass_items<K>()
                 ? (gd ? launch_pass<K, 1, 512, true>(c, hp, P, hp.pb()) : launch_pass<K, 1, 512, false>(c, hp, P, hp.pb()))
                 : (gd ? launch_pass<K, 1, 1024, true>(c, hp, P, hp.pb()) : launch_pass<K, 1, 1024, false>(c, hp, P, hp.pb()));
    if (rc) return rc;
    mark(c, 3);
    return HJ_OK;
  }
  mark(c, 0);
  if (!chunk) {
    CUDA_TRY(c, cudaMemsetAsync(P.counters, 0, hp.zero_bytes, st));  // the zeroed region starts at o_counters = 0
  } else {  // streaming S chunk: keep R's counts and the accumulated results
    CUDA_TRY(c, cudaMemsetAsync((char*)c->meta.p + hp.o_counters, 0, 64, st));
    CUDA_TRY(c, cudaMemsetAsync((char*)c->meta.p + hp.o_cnt[1], 0, (size_t)4 << hp.qbits(), st));
  }
  if (hp.mode != PLAN_RECV) {
    const bool smem = hp.qbits() <= 16;
    const bool c32 = hp.qbits() <= 15;  // 16 bins: packed 16-bit counters (128 KB)
    const size_t sm = smem ? (c32 ? ((size_t)4 << hp.qbits()) : ((size_t)2 << hp.qbits())) : 0;
    const unsigned long long nR = P.rel[0].n, nS = P.rel[1].n;
    const void* f = smem ? (gd ? (const void*)k_hist<K, true, true> : (const void*)k_hist<K, true, false>)
                         : (const void*)k_hist<K, false, false>;
    int g = std::max(2, grid_for(c, f, HIST_NT, sm, (nR + nS + 4095) / 4096 + 2));
    // blocks split proportionally to the relation sizes (at least one each)
    uint32_t gr = (uint32_t)((double)g * (double)nR / (double)std::max<unsigned long long>(nR + nS, 1) + 0.5);
    gr = std::min<uint32_t>(std::max<uint32_t>(gr, 1), (uint32_t)g - 1);
    if (nR == 0) gr = 0;  // streaming S chunk: every block counts S
    if (smem && c32 && gd) k_hist<K, true, true, true><<<g, HIST_NT, sm, st>>>(P, gr);
    else if (smem && c32) k_hist<K, true, false, true><<<g, HIST_NT, sm, st>>>(P, gr);
    else if (smem && gd) k_hist<K, true, true, false><<<g, HIST_NT, sm, st>>>(P, gr);
    else if (smem) k_hist<K, true, false, false><<<g, HIST_NT, sm, st>>>(P, gr);
    else if (gd) k_hist<K, false, true><<<g, HIST_NT, 0, st>>>(P, gr);
    else k_hist<K, false, false><<<g, HIST_NT, 0, st>>>(P, gr);
    CUDA_TRY(c, cudaGetLastError());
    c->launches += 1;
  } else if (int rc = launch_hist_recv<K>(c, hp, P)) {  // exchange receiver: its own histogram
    return rc;
  }
  mark(c, 1);
  if (int rc = launch_plan(c, hp, P)) return rc;
  mark(c, 2);
  if (stage == 1) return HJ_OK;
  if (hp.mode != PLAN_RECV) {
    int rc = hp.tile == 512 * pass_items<K>()
                 ? (gd ? launch_pass<K, 1, 512, true>(c, hp, P, hp.pb()) : launch_pass<K, 1, 512, false>(c, hp, P, hp.pb()))
                 : (gd ? launch_pass<K, 1, 1024, true>(c, hp, P, hp.pb()) : launch_pass<K, 1, 1024, false>(c, hp, P, hp.pb()));
    if (rc) return rc;
  }
  mark(c, 3);
  return HJ_OK;
}

// a3 / a4: one partition pass (launch shape per pass and width).
template <typename K, int MODE, bool GD, int CW, bool BC = false>
int launch_pass_ws(Ctx* c, const HostPlan& hp, const Plan& P, int fanout_bits) {
  using S = WsShape<K, CW>;
  const void* f = (const void*)k_pass_ws<K, MODE, GD, CW, BC>;
  const size_t sm = S::smem(fanout_bits);
  const unsigned long long tile = S::TILE;
  Plan Q = P;
  Q.C2 = (uint32_t)tile;
  unsigned long long units = MODE == 1 ? (P.rel[0].n + tile - 1) / tile + (P.rel[1].n + tile - 1) / tile
                                       : (P.rel[0].n + P.rel[1].n) / tile + 2ull * hp.npieces() + 2;
  if (BC && MODE == 2) units = (P.rel[0].n + P.rel[1].n) / tile + P.bc_rel[0].nbmax1 + P.bc_rel[1].nbmax1 + 2;
  if (MODE == 1) {
    Q.tiles1[0] = (P.rel[0].n + tile - 1) / tile;
    Q.tiles1[1] = (P.rel[1].n + tile - 1) / tile;
  }
  const int g = grid_for(c, f, WS_NT, sm, units);
  CUDA_TRY(c, launch_k(c, k_pass_ws<K, MODE, GD, CW, BC>, g, WS_NT, sm, Q, fanout_bits));
  CUDA_TRY(c, cudaGetLastError());
  c->launches += 1;
  return HJ_OK;
}

template <typename K, int MODE, int NT, bool GD, bool BC>
int launch_pass(Ctx* c, const HostPlan& hp, const Plan& P, int fanout_bits) {
  constexpr int IT = pass_items<K>();
  if constexpr (BC && !GD) {
    // pass 2 keeps the pass-1 bucket list in static shared memory (32 KB): fan-out <= 2^8
    if (use_ws(c, fanout_bits) && (MODE == 1 ? hp.tile : hp.C2) == ws_tile(c) && (MODE == 1 || fanout_bits <= 8))
      return launch_pass_ws<K, MODE, GD, 20, true>(c, hp, P, fanout_bits);
  }
  if (!BC && use_ws(c, fanout_bits) && (MODE == 1 ? hp.tile : hp.C2) == ws_tile(c)) {
    // warp-specialized pipeline: one 1024-thread block per SM
#define WS_LAUNCH_CASE(N) \
    if (ws_cw(c) == N) return launch_pass_ws<K, MODE, GD, N>(c, hp, P, fanout_bits);
    WS_CWS(WS_LAUNCH_CASE)
#undef WS_LAUNCH_CASE
  }
  const int mask = c->opt_pass_variant > 0 ? (int)c->opt_pass_variant - 1 : (c->key_bytes == 8 ? 1 : 0);
  if (NT == 1024 && ((mask >> (MODE - 1)) & 1) && (1 << fanout_bits) <= 512) {
    const void* f2 = (const void*)k_pass<K, MODE, 512, 2 * IT, GD, BC, false>;
    const size_t sm2 = (size_t)NT * IT * sizeof(typename Tup<K>::T) + ((size_t)1 << fanout_bits) * 24 + 16;
    const unsigned long long tile2 = (unsigned long long)NT * IT;
    Plan Q = P;
    Q.C2 = (uint32_t)tile2;
    if (c->opt_pass_l2pf == 2) Q.pass_l2pf = 1;
    unsigned long long units = MODE == 1 ? (P.rel[0].n + tile2 - 1) / tile2 + (P.rel[1].n + tile2 - 1) / tile2
                                         : (P.rel[0].n + P.rel[1].n) / tile2 + 2ull * hp.npieces() + 2;
    if (BC && MODE == 2) units = (P.rel[0].n + P.rel[1].n) / tile2 + P.bc_rel[0].nbmax1 + P.bc_rel[1].nbmax1 + 2;
    if (MODE == 1) {
      Q.tiles1[0] = (P.rel[0].n + tile2 - 1) / tile2;
      Q.tiles1[1] = (P.rel[1].n + tile2 - 1) / tile2;
    }
    int g = grid_for(c, f2, 512, sm2, units);
    k_pass<K, MODE, 512, 2 * IT, GD, BC, false><<<g, 512, sm2, c->stream>>>(Q, fanout_bits);
    CUDA_TRY(c, cudaGetLastError());
    c->launches += 1;
    return HJ_OK;
  }
  const void* f = (const void*)k_pass<K, MODE, NT, IT, GD, BC>;
  const size_t sm = (size_t)NT * IT * sizeof(typename Tup<K>::T) + ((size_t)1 << fanout_bits) * 24 + 16;
  const unsigned long long tile = (unsigned long long)NT * IT;
  // units: pass 1 = tiles; pass 2 = at most n / tile + pieces per relation
  Plan Q = P;
  Q.C2 = (uint32_t)tile;
  unsigned long long units = MODE == 1 ? (P.rel[0].n + tile - 1) / tile + (P.rel[1].n + tile - 1) / tile
                                       : (P.rel[0].n + P.rel[1].n) / tile + 2ull * hp.npieces() + 2;
  if (BC && MODE == 2) units = (P.rel[0].n + P.rel[1].n) / tile + P.bc_rel[0].nbmax1 + P.bc_rel[1].nbmax1 + 2;
  if (MODE == 1) {
    Q.tiles1[0] = (P.rel[0].n + tile - 1) / tile;
    Q.tiles1[1] = (P.rel[1].n + tile - 1) / tile;
  }
  int g = grid_for(c, f, NT, sm, units);
  k_pass<K, MODE, NT, IT, GD, BC><<<g, NT, sm, c->stream>>>(Q, fanout_bits);
  CUDA_TRY(c, cudaGetLastError());
  c->launches += 1;
  return HJ_OK;
}

// a4: pass 2 over the pass-1 pieces. Event 4.
template <typename K>
int launch_pass2(Ctx* c, const HostPlan& hp, const Plan& P) {
  int rc = hp.C2 == (uint32_t)(512 * pass_items<K>()) ? launch_pass<K, 2, 512, false>(c, hp, P, hp.b2)
                                                       : launch_pass<K, 2, 1024, false>(c, hp, P, hp.b2);
  if (rc) return rc;
  mark(c, 4);
  return HJ_OK;
}

template <typename K, int V, bool F2>
int launch_join_f(Ctx* c, const HostPlan& hp, const Plan& P, bool mat) {
  constexpr JoinShape S = JOIN_SHAPES[V];
  cudaStream_t st = c->stream;
  const void* f = mat ? (const void*)k_join<K, S.nt, S.spt, true, S.minb, S.rbuf, S.h16, S.pf, S.l2pf, S.spf, F2, S.bf>
                      : (const void*)k_join<K, S.nt, S.spt, false, S.minb, S.rbuf, S.h16, S.pf, S.l2pf, S.spf, F2, S.bf>;
  int g = grid_for(c, f, S.nt + 32, hp.join_smem, 1ull << 40);
  if (mat)
    CUDA_TRY(c, launch_k(c, k_join<K, S.nt, S.spt, true, S.minb, S.rbuf, S.h16, S.pf, S.l2pf, S.spf, F2, S.bf>, g,
                         S.nt + 32, hp.join_smem, P));
  else
    CUDA_TRY(c, launch_k(c, k_join<K, S.nt, S.spt, false, S.minb, S.rbuf, S.h16, S.pf, S.l2pf, S.spf, F2, S.bf>, g,
                         S.nt + 32, hp.join_smem, P));
  CUDA_TRY(c, cudaGetLastError());
  return HJ_OK;
}

// the cheaper slot hash (slot_of2): 8-byte keys always, 4-byte keys when the two-term fold still
// covers every key bit above the radix field
template <typename K, int V>
int launch_join_v(Ctx* c, const HostPlan& hp, const Plan& P, bool mat) {
  if (sizeof(K) == 8 || P.H.nfold <= 1) return launch_join_f<K, V, true>(c, hp, P, mat);
  return launch_join_f<K, V, sizeof(K) == 8>(c, hp, P, mat);
}

template <typename K>
int launch_join(Ctx* c, const HostPlan& hp, const Plan& P, bool mat) {
  int rc;
  if (c->opt_join_algo == 1) {  // ballot nested-loop co-partition join (Listing 1)
    const size_t sm = (size_t)hp.CR * 2 * sizeof(K);
    const void* f = mat ? (const void*)k_join_nlj<K, 256, true> : (const void*)k_join_nlj<K, 256, false>;
    const int g = grid_for(c, f, 256, sm, 1ull << 40);
    if (mat) k_join_nlj<K, 256, true><<<g, 256, sm, c->stream>>>(P);
    else k_join_nlj<K, 256, false><<<g, 256, sm, c->stream>>>(P);
    CUDA_TRY(c, cudaGetLastError());
    mark(c, 5);
    c->launches += 1;
    return HJ_OK;
  }
  switch (join_variant(c, mat)) {
    case 1: rc = launch_join_v<K, 1>(c, hp, P, mat); break;
    case 2: rc = launch_join_v<K, 2>(c, hp, P, mat); break;
    case 3: rc = launch_join_v<K, 3>(c, hp, P, mat); break;
    case 4: rc = launch_join_v<K, 4>(c, hp, P, mat); break;
    case 5: rc = launch_join_v<K, 5>(c, hp, P, mat); break;
    case 6: rc = launch_join_v<K, 6>(c, hp, P, mat); break;
    case 7: rc = launch_join_v<K, 7>(c, hp, P, mat); break;
    case 8: rc = launch_join_v<K, 8>(c, hp, P, mat); break;


    default: rc = launch_join_v<K, 0>(c, hp, P, mat); break;
  }
  if (rc) return rc;
  mark(c, 5);
  c->launches += 1;
  return HJ_OK;
}

int prepare(Ctx* c, HostPlan& hp, unsigned long long nR, unsigned long long nS, int radix_bits, bool mat, int g = 0,
            int nsrc = 1, int mode = PLAN_FULL, unsigned long long nR_est = 0) {
  int rc = make_plan(c, hp, nR, nS, radix_bits, mat, g, nsrc, mode, nR_est);
  if (rc) return rc;
  const size_t tb = (size_t)c->key_bytes + c->pay_bytes;
  const unsigned long long ns[2] = {nR, nS};
  for (int r = 0; r < 2; ++r) {
    if (mode == PLAN_FULL && (rc = ensure(c, c->t1[r], ns[r] * tb))) return rc;
    if (mode != PLAN_SEND && (rc = ensure(c, c->t2[r], ns[r] * tb + 64))) return rc;  // +64: aligned bulk-copy tail
  }
  if ((rc = ensure(c, c->meta, hp.meta_bytes))) return rc;
  if (mat) {
    unsigned long long cap = c->opt_out_cap > 0 ? (unsigned long long)c->opt_out_cap : std::max<unsigned long long>(nS, 1 << 20);
    if (out_short(c, cap)) {
      if ((rc = ensure(c, c->out_r, cap * c->pay_bytes))) return rc;
      if ((rc = ensure(c, c->out_s, cap * c->pay_bytes))) return rc;
    }
  }
  return HJ_OK;
}

// Join phase + result readback shared by hj_join and hj_join_received.
int finish_join(Ctx* c, const HostPlan& hp, Plan& P, bool mat, hj_result* res, const XdJoin* xd = nullptr) {
  cudaStream_t st = c->stream;
  const bool timing = c->opt_timing != 0;
  int rc = c->key_bytes == 4 ? launch_join<uint32_t>(c, hp, P, mat) : launch_join<uint64_t>(c, hp, P, mat);
  if (rc) return rc;
  unsigned long long* h = c->async ? c->async->h : (unsigned long long*)c->h_res;
  if (xd) {  // hj_xd_join: phase C (results of every rank summed on the device) before the readback
    k_xd_results<<<1, XD_MAX, 0, st>>>(*xd);
    CUDA_TRY(c, cudaGetLastError());
    c->launches += 1;
  }
  CUDA_TRY(c, cudaMemcpyAsync(h, P.results, 4 * sizeof(unsigned long long), cudaMemcpyDeviceToHost, st));
  CUDA_TRY(c, cudaMemcpyAsync(h + 4, P.ist + (1ull << hp.B), sizeof(uint32_t), cudaMemcpyDeviceToHost, st));
  if (xd) CUDA_TRY(c, cudaMemcpyAsync(h + 6, P.results + 4, 3 * sizeof(unsigned long long), cudaMemcpyDeviceToHost, st));
  h[5] = 0;
  if (P.mode == PLAN_RECV)
    CUDA_TRY(c, cudaMemcpyAsync(h + 5, P.counters + CNT_BAD_COUNTS, sizeof(uint32_t), cudaMemcpyDeviceToHost, st));
  if (c->async) {  // hj_join_async: the readback is enqueued; complete_pending() finishes the call
    Pending& q = *c->async;
    CUDA_TRY(c, cudaEventRecord(c->ev[6], st));
    q.B = hp.B;
    q.mat = mat;
    q.bc = P.bc != 0;
    q.recv = P.mode == PLAN_RECV;
    q.timing = timing;
    q.out_cap = P.out_cap;
    q.out_r = c->out_r.p;
    q.out_s = c->out_s.p;
    q.launches = c->launches;
    return HJ_OK;
  }
  if (timing) CUDA_TRY(c, cudaEventRecord(c->ev[6], st));
  CUDA_TRY(c, cudaStreamSynchronize(st));
  if (P.bc && h[RES_BC_OVERFLOW]) return fail(c, HJ_ERR_CUDA, "bucket pool overflow (pool bound violated)");
  if ((uint32_t)h[5])
    return fail(c, HJ_ERR_INVALID, "received count rows describe more tuples than the received buffers hold");
  unsigned long long matches = h[RES_MATCHES];
  if (mat && matches > P.out_cap) {
    // materialization overflow (reading S11): never overwrite -- grow to the exact size and re-run
    // only the join; with a caller workspace the caller grows it (HJ_ERR_WORKSPACE, exact count)
    if (c->use_ws) {
      memset(res, 0, sizeof *res);
      res->matches = matches;
      return fail(c, HJ_ERR_WORKSPACE, "materialized output needs %llu pairs (capacity %llu): set "
                  "HJ_OPT_OUT_CAPACITY >= matches and resize the workspace", matches, P.out_cap);
    }
    if ((rc = ensure(c, c->out_r, matches * c->pay_bytes))) return rc;
    if ((rc = ensure(c, c->out_s, matches * c->pay_bytes))) return rc;
    P.out_r = c->out_r.p;
    P.out_s = c->out_s.p;
    P.out_cap = matches;
    CUDA_TRY(c, cudaMemsetAsync(P.results, 0, 4 * sizeof(unsigned long long), st));
    CUDA_TRY(c, cudaMemsetAsync(P.counters, 0, 8 * sizeof(uint32_t), st));
    rc = c->key_bytes == 4 ? launch_join<uint32_t>(c, hp, P, mat) : launch_join<uint64_t>(c, hp, P, mat);
    if (rc) return rc;
    CUDA_TRY(c, cudaMemcpyAsync(h, P.results, 4 * sizeof(unsigned long long), cudaMemcpyDeviceToHost, st));
    if (timing) CUDA_TRY(c, cudaEventRecord(c->ev[6], st));
    CUDA_TRY(c, cudaStreamSynchronize(st));
    matches = h[RES_MATCHES];
  }
  memset(res, 0, sizeof *res);
  res->matches = matches;
  res->checksum = h[RES_CHECKSUM];
  res->n_items = (uint32_t)h[4];
  res->radix_bits = hp.B;
  res->passes = hp.B >= 2 ? 2 : (hp.B == 1 ? 1 : 0);
  if (mat) {
    res->r_pay_out = c->out_r.p;
    res->s_pay_out = c->out_s.p;
  }
  res->kernels = c->launches;
  if (timing) {
    cudaEventElapsedTime(&res->ms_total, c->ev[0], c->ev[6]);
    cudaEventElapsedTime(&res->ms_partition, c->ev[0], c->ev[4]);
    cudaEventElapsedTime(&res->ms_join, c->ev[4], c->ev[6]);
    for (int k = 0; k < 5; ++k) cudaEventElapsedTime(&res->ms_kernel[k], c->ev[k], c->ev[k + 1]);
    cudaGetLastError();  // a phase that recorded no event (e.g. skipped) must not fail the next call
  }
  return HJ_OK;
}

// HJ_OPT_JOIN_ALGO = 2: the non-partitioned GPU hash join (device-memory chained table; the
// paper's Fig. 8 baseline). No histogram, no passes: build R, probe S.
template <typename K>
int run_join_np(Ctx* c, const void* Rk, const void* Rp, unsigned long long nR, const void* Sk, const void* Sp,
                unsigned long long nS, bool mat, hj_result* res) {
  HostPlan hp;
  int rc = make_plan(c, hp, nR, nS, 0, mat);
  if (rc) return rc;
  const int lg = std::max(1, ilog2_ceil(nR));
  if ((rc = ensure(c, c->meta, hp.meta_bytes)) || (rc = ensure(c, c->np_heads, (size_t)4 << lg)) ||
      (rc = ensure(c, c->np_next, nR * 4)))
    return rc;
  unsigned long long cap = c->opt_out_cap > 0 ? (unsigned long long)c->opt_out_cap : std::max<unsigned long long>(nS, 1 << 20);
  if (mat && out_short(c, cap) &&
      ((rc = ensure(c, c->out_r, cap * c->pay_bytes)) || (rc = ensure(c, c->out_s, cap * c->pay_bytes))))
    return rc;
  if (c->dry) return HJ_OK;
  Plan P = device_plan(c, hp, Rk, Rp, nR, Sk, Sp, nS);
  cudaStream_t st = c->stream;
  c->launches = 0;
  for (int attempt = 0; attempt < 2; ++attempt) {
    mark(c, 0);
    CUDA_TRY(c, cudaMemsetAsync(c->meta.p, 0, hp.zero_bytes, st));
    CUDA_TRY(c, cudaMemsetAsync(c->np_heads.p, 0xff, (size_t)4 << lg, st));
    for (int k = 1; k <= 4; ++k) mark(c, k);
    const int g = 4 * c->num_sms;
    k_np_build<K><<<g, 512, 0, st>>>((const K*)Rk, nR, (uint32_t*)c->np_heads.p, (uint32_t*)c->np_next.p, lg);
    if (mat)
      k_np_probe<K, true><<<g, 512, 0, st>>>(P, (const K*)Rk, (const K*)Rp, (const K*)Sk, (const K*)Sp, nS,
                                              (const uint32_t*)c->np_heads.p, (const uint32_t*)c->np_next.p, lg);
    else
      k_np_probe<K, false><<<g, 512, 0, st>>>(P, (const K*)Rk, (const K*)Rp, (const K*)Sk, (const K*)Sp, nS,
                                               (const uint32_t*)c->np_heads.p, (const uint32_t*)c->np_next.p, lg);
    CUDA_TRY(c, cudaGetLastError());
    c->launches += 2;
    mark(c, 5);
    unsigned long long* h = (unsigned long long*)c->h_res;
    CUDA_TRY(c, cudaMemcpyAsync(h, P.results, 4 * sizeof(unsigned long long), cudaMemcpyDeviceToHost, st));
    mark(c, 6);
    CUDA_TRY(c, cudaStreamSynchronize(st));
    if (mat && h[RES_MATCHES] > P.out_cap && attempt == 0) {  // grow and re-run (reading S11)
      if (c->use_ws) {
        memset(res, 0, sizeof *res);
        res->matches = h[RES_MATCHES];
        return fail(c, HJ_ERR_WORKSPACE, "materialized output needs %llu pairs: set HJ_OPT_OUT_CAPACITY and resize "
                    "the workspace", h[RES_MATCHES]);
      }
      if ((rc = ensure(c, c->out_r, h[RES_MATCHES] * c->pay_bytes)) ||
          (rc = ensure(c, c->out_s, h[RES_MATCHES] * c->pay_bytes)))
        return rc;
      P.out_r = c->out_r.p;
      P.out_s = c->out_s.p;
      P.out_cap = h[RES_MATCHES];
      continue;
    }
    memset(res, 0, sizeof *res);
    res->matches = h[RES_MATCHES];
    res->checksum = h[RES_CHECKSUM];
    res->kernels = c->launches;
    if (mat) {
      res->r_pay_out = c->out_r.p;
      res->s_pay_out = c->out_s.p;
    }
    if (c->opt_timing) {
      cudaEventElapsedTime(&res->ms_total, c->ev[0], c->ev[6]);
      cudaEventElapsedTime(&res->ms_join, c->ev[4], c->ev[6]);
      for (int k = 0; k < 5; ++k) cudaEventElapsedTime(&res->ms_kernel[k], c->ev[k], c->ev[k + 1]);
    }
    return HJ_OK;
  }
  return HJ_OK;
}

// Wait for the oldest pending hj_join_async call and fill its result (as finish_join's tail).
// Post-hoc failures (bucket pool, received rows, output capacity) are reported here.
int complete_pending(Ctx* c) {
  Pending& q = c->pend[c->pend_head];
  c->pend_head = (c->pend_head + 1) % MAX_PENDING;
  c->pend_n--;
  hj_result* res = q.res;
  const unsigned long long* h = q.h;
  CUDA_TRY(c, cudaEventSynchronize(q.ev[6]));
  memset(res, 0, sizeof *res);
  if (q.bc && h[RES_BC_OVERFLOW]) return fail(c, HJ_ERR_CUDA, "bucket pool overflow (pool bound violated)");
  if (q.recv && (uint32_t)h[5])
    return fail(c, HJ_ERR_INVALID, "received count rows describe more tuples than the received buffers hold");
  res->matches = h[RES_MATCHES];
  if (q.mat && res->matches > q.out_cap)  // no re-run: later calls have reused the buffers
    return fail(c, HJ_ERR_WORKSPACE, "materialized output needs %llu pairs (capacity %llu): set "
                "HJ_OPT_OUT_CAPACITY >= matches and call again", res->matches, q.out_cap);
  res->checksum = h[RES_CHECKSUM];
  res->n_items = (uint32_t)h[4];
  res->radix_bits = q.B;
  res->passes = q.B >= 2 ? 2 : (q.B == 1 ? 1 : 0);
  if (q.mat) {
    res->r_pay_out = q.out_r;
    res->s_pay_out = q.out_s;
  }
  res->kernels = q.launches;
  if (q.timing) {
    cudaEventElapsedTime(&res->ms_total, q.ev[0], q.ev[6]);
    cudaEventElapsedTime(&res->ms_partition, q.ev[0], q.ev[4]);
    cudaEventElapsedTime(&res->ms_join, q.ev[4], q.ev[6]);
    for (int k = 0; k < 5; ++k) cudaEventElapsedTime(&res->ms_kernel[k], q.ev[k], q.ev[k + 1]);
    cudaGetLastError();
  }
  return HJ_OK;
}

// Complete every pending call in issue order; the first failure's code (its message stays in
// c->err unless a later one overwrites it -- the first is kept).
int drain_pending(Ctx* c) {
  int first = HJ_OK;
  std::string msg;
  while (c->pend_n > 0) {
    const int rc = complete_pending(c);
    if (rc && first == HJ_OK) {
      first = rc;
      msg = c->err;
    }
  }
  if (first) c->err = msg;
  return first;
}

// One-shot graph path (HJ_OPT_GRAPH): kernels + result readback captured from the ctx stream;
// timing events are recorded around the replay only (ms_kernel stays 0).
int run_join_graph_on(Ctx* c, HostPlan& hp, Plan& P, bool mat, const unsigned long long* key, hj_result* res);

// The capture and replays run on the ctx-owned stream (the caller's may be the legacy default
// stream, which cannot be captured), ordered after the caller's stream by an event; the call is
// synchronous, so later work on the caller's stream sees the results.
int run_join_graph(Ctx* c, HostPlan& hp, Plan& P, bool mat, const unsigned long long* key, hj_result* res) {
  cudaStream_t caller = c->stream;
  if (caller != c->own_stream) {
    CUDA_TRY(c, cudaEventRecord(c->ev[7], caller));
    CUDA_TRY(c, cudaStreamWaitEvent(c->own_stream, c->ev[7], 0));
  }
  c->stream = c->own_stream;
  const int rc = run_join_graph_on(c, hp, P, mat, key, res);
  c->stream = caller;
  return rc;
}

int run_join_graph_on(Ctx* c, HostPlan& hp, Plan& P, bool mat, const unsigned long long* key, hj_result* res) {
  cudaStream_t st = c->stream;
  unsigned long long* h = (unsigned long long*)c->h_res;
  if (!c->graph || memcmp(key, c->graph_key, sizeof c->graph_key) != 0) {
    if (c->graph) cudaGraphExecDestroy(c->graph);
    c->graph = nullptr;
    // no event records inside the capture: as external event-record nodes they cost the replay
    // its gain (c3: 2.69 -> 2.74-2.89 ms/call, measured), so a replay reports ms_total only
    const int64_t timing = c->opt_timing;
    c->opt_timing = 0;
    c->launches = 0;
    CUDA_TRY(c, cudaStreamBeginCapture(st, cudaStreamCaptureModeThreadLocal));
    c->capturing = true;
    int rc = c->key_bytes == 4 ? launch_front<uint32_t>(c, hp, P) : launch_front<uint64_t>(c, hp, P);
    if (!rc) rc = c->key_bytes == 4 ? launch_pass2<uint32_t>(c, hp, P) : launch_pass2<uint64_t>(c, hp, P);
    if (!rc) rc = c->key_bytes == 4 ? launch_join<uint32_t>(c, hp, P, mat) : launch_join<uint64_t>(c, hp, P, mat);
    if (!rc && cudaMemcpyAsync(h, P.results, 4 * sizeof(unsigned long long), cudaMemcpyDeviceToHost, st) != cudaSuccess)
      rc = fail(c, HJ_ERR_CUDA, "capture: results copy");
    if (!rc && cudaMemcpyAsync(h + 4, P.ist + (1ull << hp.B), sizeof(uint32_t), cudaMemcpyDeviceToHost, st) != cudaSuccess)
      rc = fail(c, HJ_ERR_CUDA, "capture: items copy");
    cudaGraph_t g = nullptr;
    cudaError_t e = cudaStreamEndCapture(st, &g);
    c->capturing = false;
    c->opt_timing = timing;
    if (rc) {
      if (g) cudaGraphDestroy(g);
      return rc;
    }
    if (e != cudaSuccess) return fail(c, HJ_ERR_CUDA, "graph capture: %s", cudaGetErrorString(e));
    e = cudaGraphInstantiate(&c->graph, g, 0);
    cudaGraphDestroy(g);
    if (e != cudaSuccess) {
      c->graph = nullptr;
      return fail(c, HJ_ERR_CUDA, "graph instantiate: %s", cudaGetErrorString(e));
    }
    memcpy(c->graph_key, key, sizeof c->graph_key);
    c->graph_launches = c->launches;
  }
  if (c->opt_timing) CUDA_TRY(c, cudaEventRecord(c->ev[0], st));
  CUDA_TRY(c, cudaGraphLaunch(c->graph, st));
  if (c->opt_timing) CUDA_TRY(c, cudaEventRecord(c->ev[6], st));
  CUDA_TRY(c, cudaStreamSynchronize(st));
  if (mat && h[RES_MATCHES] > P.out_cap) {  // overflow: drop the graph, redo on the normal path
    cudaGraphExecDestroy(c->graph);
    c->graph = nullptr;
    c->launches = 0;
    int rc = c->key_bytes == 4 ? launch_front<uint32_t>(c, hp, P) : launch_front<uint64_t>(c, hp, P);
    if (!rc) rc = c->key_bytes == 4 ? launch_pass2<uint32_t>(c, hp, P) : launch_pass2<uint64_t>(c, hp, P);
    return rc ? rc : finish_join(c, hp, P, mat, res);
  }
  memset(res, 0, sizeof *res);
  res->matches = h[RES_MATCHES];
  res->checksum = h[RES_CHECKSUM];
  res->n_items = (uint32_t)h[4];
  res->radix_bits = hp.B;
  res->passes = hp.B >= 2 ? 2 : (hp.B == 1 ? 1 : 0);
  res->kernels = c->graph_launches;
  if (mat) {
    res->r_pay_out = c->out_r.p;
    res->s_pay_out = c->out_s.p;
  }
  if (c->opt_timing) cudaEventElapsedTime(&res->ms_total, c->ev[0], c->ev[6]);
  return HJ_OK;
}

// HJ_OPT_PARTITIONER = 1: the paper's histogram-free bucket-chain partitioner (NEXT-1,
// hj_bucket.cuh). Pool sizes are the proven bounds of hj_bucket.cuh: a closed bucket holds >= cap
// tuples, so n / cap + min(partitions, n) buckets suffice per relation and pass.
template <typename K>
int run_join_bc(Ctx* c, const void* Rk, const void* Rp, unsigned long long nR, const void* Sk, const void* Sp,
                unsigned long long nS, int radix_bits, bool mat, hj_result* res) {
  HostPlan hp;
  int rc = make_plan(c, hp, nR, nS, radix_bits, mat);
  if (rc) return rc;
  if ((rc = ensure(c, c->meta, hp.meta_bytes))) return rc;
  if (mat) {
    unsigned long long cap = c->opt_out_cap > 0 ? (unsigned long long)c->opt_out_cap : std::max<unsigned long long>(nS, 1 << 20);
    if (out_short(c, cap) &&
        ((rc = ensure(c, c->out_r, cap * c->pay_bytes)) || (rc = ensure(c, c->out_s, cap * c->pay_bytes))))
      return rc;
  }
  Plan P = device_plan(c, hp, Rk, Rp, nR, Sk, Sp, nS);
  P.bc = 1;
  P.ist2 = nullptr;  // the bucket-chain planner makes no swapped items
  const size_t tb = sizeof(typename Tup<K>::T);
  const unsigned long long ns[2] = {nR, nS}, F1 = 1ull << hp.b1, np = 1ull << hp.B;
  const uint32_t tile1 = (uint32_t)hp.tile, C2 = hp.C2;
  // metadata layout: zeroed part first (states, pass-2 fills, slice counts)
  size_t o = 0, o_st1[2], o_st2[2], o_fill2[2], o_nsl[2], o_fill1[2], o_part1[2], o_part2[2], o_sl[2],
         o_sst[2], o_scur[2];
  auto take = [&](size_t bytes) {
    size_t r = o;
    o = align_up(o + bytes, 256);
    return r;
  };
  // capacities: 2x the mean partition (uniform inputs never close a bucket; a skewed partition
  // closes one per cap tuples), at least 4 tiles in pass 1; stride = cap + tile (closing run)
  auto cap_for = [](unsigned long long mean, uint32_t tile, unsigned long long min_tiles) {
    const unsigned long long t = std::max<unsigned long long>(min_tiles, (2 * mean + tile - 1) / tile);
    return (uint32_t)std::min<unsigned long long>(t * tile, 1ull << 30);
  };
  for (int r = 0; r < 2; ++r) {
    BcRel& B = P.bc_rel[r];
    B.cap1 = cap_for((ns[r] + F1 - 1) / F1, tile1, 4);
    B.bsz1 = (unsigned long long)B.cap1 + tile1;
    B.cap2 = cap_for((ns[r] + np - 1) / np, C2, 1);
    B.bsz2 = (unsigned long long)B.cap2 + C2;
    B.np1 = (uint32_t)F1;
    B.np2 = (uint32_t)np;
    B.nbmax1 = (uint32_t)(ns[r] / B.cap1 + F1 + 1);
    if (B.nbmax1 + 5 > BC_MAX_NB1) return fail(c, HJ_ERR_INVALID, "bucket chains: %u pass-1 buckets", B.nbmax1);
    // pass 2 grows a hot partition's regions up to 16 buckets (as long as a region's fill stays
    // below 2^30), bound 2n / cap2 + np + 1 (hj_bucket.cuh)
    B.lg2max = 0;
    while (B.lg2max < 4 && (B.bsz2 << (B.lg2max + 1)) <= (1ull << 30)) ++B.lg2max;
    B.nbmax2 = (uint32_t)((B.lg2max ? 2 : 1) * (ns[r] / B.cap2) + np + 1);
    B.csl = r == 0 ? hp.CR : hp.CS;
    o_st1[r] = take(F1 * 8);
    o_st2[r] = take(np * 8);
    o_nsl[r] = take(np * 4);
  }
  const size_t zero_bytes = o;
  for (int r = 0; r < 2; ++r) {
    const BcRel& B = P.bc_rel[r];
    o_fill1[r] = take((size_t)B.nbmax1 * 4);
    o_part1[r] = take((size_t)B.nbmax1 * 4);
    o_part2[r] = take((size_t)B.nbmax2 * 4);
    o_fill2[r] = take((size_t)B.nbmax2 * 4);
    o_sl[r] = take((ns[r] / B.csl + B.nbmax2 + 1) * 16);
    o_sst[r] = take((np + 1) * 4);
    o_scur[r] = take(np * 4);
  }
  if ((rc = ensure(c, c->bc_meta, o))) return rc;
  for (int r = 0; r < 2; ++r) {
    BcRel& B = P.bc_rel[r];
    if ((rc = ensure(c, c->bc_pool1[r], (size_t)B.nbmax1 * B.bsz1 * tb))) return rc;
    if ((rc = ensure(c, c->bc_pool2[r], (size_t)B.nbmax2 * B.bsz2 * tb))) return rc;
    if (c->dry) continue;
    char* m = (char*)c->bc_meta.p;
    B.pool1 = c->bc_pool1[r].p;
    B.pool2 = c->bc_pool2[r].p;
    B.st1 = (unsigned long long*)(m + o_st1[r]);
    B.st2 = (unsigned long long*)(m + o_st2[r]);
    B.fill1 = (uint32_t*)(m + o_fill1[r]);
    B.part1 = (uint32_t*)(m + o_part1[r]);
    B.fill2 = (uint32_t*)(m + o_fill2[r]);
    B.part2 = (uint32_t*)(m + o_part2[r]);
    B.sl = (uint4*)(m + o_sl[r]);
    B.nsl = (uint32_t*)(m + o_nsl[r]);
    B.sst = (uint32_t*)(m + o_sst[r]);
    B.scur = (uint32_t*)(m + o_scur[r]);
    P.rel[r].t2 = B.pool2;  // the join reads slices of the pass-2 pool
  }
  if (c->dry) return HJ_OK;
  cudaStream_t st = c->stream;
  c->launches = 0;
  mark(c, 0);
  CUDA_TRY(c, cudaMemsetAsync(c->meta.p, 0, hp.zero_bytes, st));
  CUDA_TRY(c, cudaMemsetAsync(c->bc_meta.p, 0, zero_bytes, st));
  mark(c, 1);  // no histogram
  mark(c, 2);  // no planner before the passes
  rc = hp.tile == 512 * pass_items<K>() ? launch_pass<K, 1, 512, false, true>(c, hp, P, hp.b1)
                                        : launch_pass<K, 1, 1024, false, true>(c, hp, P, hp.b1);
  if (rc) return rc;
  mark(c, 3);
  rc = C2 == (uint32_t)(512 * pass_items<K>()) ? launch_pass<K, 2, 512, false, true>(c, hp, P, hp.b2)
                                               : launch_pass<K, 2, 1024, false, true>(c, hp, P, hp.b2);
  if (rc) return rc;
  const unsigned long long idx = np + std::max(P.bc_rel[0].nbmax2, P.bc_rel[1].nbmax2);
  const int gc = (int)std::min<unsigned long long>((idx + 255) / 256, 4ull * c->num_sms);
  k_bc_plan<<<(unsigned)((np + 1023) / 1024), 1024, 0, st>>>(P);
  k_bc_slices<<<gc, 256, 0, st>>>(P);
  CUDA_TRY(c, cudaGetLastError());
  c->launches += 2;
  mark(c, 4);
  return finish_join(c, hp, P, mat, res);
}

int run_join(Ctx* c, const void* Rk, const void* Rp, unsigned long long nR, const void* Sk, const void* Sp,
             unsigned long long nS, int radix_bits, int out_mode, hj_result* res) {
  const bool mat = out_mode == HJ_OUT_MATERIALIZE;
  if (c->opt_join_algo == 2)
    return c->key_bytes == 4 ? run_join_np<uint32_t>(c, Rk, Rp, nR, Sk, Sp, nS, mat, res)
                             : run_join_np<uint64_t>(c, Rk, Rp, nR, Sk, Sp, nS, mat, res);
  if (c->opt_partitioner == 1)
    return c->key_bytes == 4 ? run_join_bc<uint32_t>(c, Rk, Rp, nR, Sk, Sp, nS, radix_bits, mat, res)
                             : run_join_bc<uint64_t>(c, Rk, Rp, nR, Sk, Sp, nS, radix_bits, mat, res);
  HostPlan hp;
  int rc = prepare(c, hp, nR, nS, radix_bits, mat);
  if (rc || c->dry) return rc;
  Plan P = device_plan(c, hp, Rk, Rp, nR, Sk, Sp, nS);
  if (c->opt_graph) {
    // every address and size the captured launch sequence bakes in (ensure() also drops the graph
    // whenever it reallocates a buffer)
    const unsigned long long key[16] = {(unsigned long long)Rk, (unsigned long long)Rp, nR, (unsigned long long)Sk,
                                        (unsigned long long)Sp, nS, (unsigned long long)hp.B * 2 + mat,
                                        (unsigned long long)c->meta.p, (unsigned long long)c->out_r.p,
                                        (unsigned long long)c->out_s.p, P.out_cap,
                                        (unsigned long long)c->t1[0].p, (unsigned long long)c->t1[1].p,
                                        (unsigned long long)c->t2[0].p, (unsigned long long)c->t2[1].p,
                                        (unsigned long long)c->opt_join_algo};
    return run_join_graph(c, hp, P, mat, key, res);
  }
  c->launches = 0;
  if ((rc = c->key_bytes == 4 ? launch_front<uint32_t>(c, hp, P) : launch_front<uint64_t>(c, hp, P))) return rc;
  if ((rc = c->key_bytes == 4 ? launch_pass2<uint32_t>(c, hp, P) : launch_pass2<uint64_t>(c, hp, P))) return rc;
  return finish_join(c, hp, P, mat, res);
}

int check_args(Ctx* c, const void* Rk, const void* Rp, unsigned long long nR, const void* Sk, const void* Sp,
               unsigned long long nS, int radix_bits, int out_mode) {
  if (out_mode != HJ_OUT_COUNT_CHECKSUM && out_mode != HJ_OUT_MATERIALIZE)
    return fail(c, HJ_ERR_INVALID, "bad out_mode %d", out_mode);
  if (radix_bits > 20) return fail(c, HJ_ERR_UNSUPPORTED, "radix_bits %d > 20", radix_bits);
  if (nR && (!Rk || !Rp)) return fail(c, HJ_ERR_INVALID, "null R column with nR > 0");
  if (nS && (!Sk || !Sp)) return fail(c, HJ_ERR_INVALID, "null S column with nS > 0");
  if (nR >= (1ull << 40) || nS >= (1ull << 40)) return fail(c, HJ_ERR_UNSUPPORTED, "relation too large");
  return HJ_OK;
}


// ---- NEXT-3: streaming join from host memory (§IV-A, §IV-C) ---------
// R is copied and partitioned once; S is copied in chunks on a copy stream into two device
// buffers (one being copied, one being processed) while the compute stream
// partitions each chunk and joins it with the resident R (the union of the chunk joins is the
// join); materialized pairs are drained to pinned host memory on a third stream as
// each chunk finishes. Falls back to the serial path if the result outgrows the
// device output buffer.
int join_host_serial(Ctx* c, const void* Rk, const void* Rp, uint64_t nR, const void* Sk, const void* Sp, uint64_t nS,
                     int radix_bits, int out_mode, hj_result* res);

int ensure_host(Ctx* c, size_t need) {
  if (c->h_out_bytes >= need) return HJ_OK;
  if (c->h_out) cudaFreeHost(c->h_out);
  c->h_out = nullptr;
  c->h_out_bytes = 0;
  if (cudaMallocHost(&c->h_out, need) != cudaSuccess) return fail(c, HJ_ERR_OOM, "pinned host alloc of %zu B", need);
  c->h_out_bytes = need;
  return HJ_OK;
}

template <typename K>
int join_host_stream(Ctx* c, const void* Rk, const void* Rp, uint64_t nR, const void* Sk, const void* Sp, uint64_t nS,
                     int radix_bits, int out_mode, uint64_t chunk, hj_result* res) {
  const bool mat = out_mode == HJ_OUT_MATERIALIZE;
  const size_t kb = c->key_bytes, pb = c->pay_bytes;
  cudaStream_t e = c->stream, t = c->h2d_stream, d = c->d2h_stream;
  cudaEvent_t ev_start = c->sev[0], ev_r = c->sev[1], ev_s[2] = {c->sev[2], c->sev[3]},
              ev_free[2] = {c->sev[4], c->sev[5]}, ev_j[2] = {c->sev[6], c->sev[7]}, ev_d = c->sev[8],
              ev_end = c->sev[9];
  HostPlan hp;
  int rc = prepare(c, hp, nR, chunk, radix_bits, mat);
  if (rc) return rc;
  const unsigned long long cap = c->opt_out_cap > 0 ? (unsigned long long)c->opt_out_cap : std::max<unsigned long long>(nS, 1 << 20);
  if (mat) {
    if ((rc = ensure(c, c->out_r, cap * pb)) || (rc = ensure(c, c->out_s, cap * pb))) return rc;
    if ((rc = ensure_host(c, 2 * cap * pb))) return rc;
  }
  if ((rc = ensure(c, c->in[0], nR * kb)) || (rc = ensure(c, c->in[1], nR * pb))) return rc;
  for (int b = 0; b < 2; ++b)
    if ((rc = ensure(c, c->sin[b][0], chunk * kb)) || (rc = ensure(c, c->sin[b][1], chunk * pb))) return rc;
  c->launches = 0;
  CUDA_TRY(c, cudaEventRecord(ev_start, t));
  // R: copy, then partition (rows a1-a4 with S empty)
  CUDA_TRY(c, cudaMemcpyAsync(c->in[0].p, Rk, nR * kb, cudaMemcpyHostToDevice, t));
  CUDA_TRY(c, cudaMemcpyAsync(c->in[1].p, Rp, nR * pb, cudaMemcpyHostToDevice, t));
  CUDA_TRY(c, cudaEventRecord(ev_r, t));
  CUDA_TRY(c, cudaStreamWaitEvent(e, ev_r, 0));
  Plan P = device_plan(c, hp, c->in[0].p, c->in[1].p, nR, nullptr, nullptr, 0);
  if ((rc = launch_front<K>(c, hp, P))) return rc;
  if ((rc = launch_pass2<K>(c, hp, P))) return rc;
  char* ho = (char*)c->h_out;
  unsigned long long* hcur = (unsigned long long*)c->h_cur;
  unsigned long long drained = 0;
  bool overflow = false;
  const uint64_t nch = (nS + chunk - 1) / chunk;
  auto drain = [&](int slot) -> int {  // host: chunk in `slot` finished -> copy its new pairs out
    CUDA_TRY(c, cudaEventSynchronize(ev_j[slot]));
    const unsigned long long cur = hcur[slot];
    if (cur > cap) overflow = true;
    if (overflow || cur <= drained) return HJ_OK;
    CUDA_TRY(c, cudaStreamWaitEvent(d, ev_j[slot], 0));
    CUDA_TRY(c, cudaMemcpyAsync(ho + drained * pb, (char*)c->out_r.p + drained * pb, (cur - drained) * pb,
                                cudaMemcpyDeviceToHost, d));
    CUDA_TRY(c, cudaMemcpyAsync(ho + (cap + drained) * pb, (char*)c->out_s.p + drained * pb, (cur - drained) * pb,
                                cudaMemcpyDeviceToHost, d));
    drained = cur;
    return HJ_OK;
  };
  for (uint64_t k = 0; k < nch; ++k) {
    const int b = (int)(k & 1);
    const uint64_t s0 = k * chunk, len = std::min<uint64_t>(chunk, nS - s0);
    // copy stream: S chunk k into buffer b once chunk k-2 has left it
    if (k >= 2) CUDA_TRY(c, cudaStreamWaitEvent(t, ev_free[b], 0));
    CUDA_TRY(c, cudaMemcpyAsync(c->sin[b][0].p, (const char*)Sk + s0 * kb, len * kb, cudaMemcpyHostToDevice, t));
    CUDA_TRY(c, cudaMemcpyAsync(c->sin[b][1].p, (const char*)Sp + s0 * pb, len * pb, cudaMemcpyHostToDevice, t));
    CUDA_TRY(c, cudaEventRecord(ev_s[b], t));
    // compute stream: partition the chunk (R skipped) and join it with R
    CUDA_TRY(c, cudaStreamWaitEvent(e, ev_s[b], 0));
    Plan Q = device_plan(c, hp, nullptr, nullptr, 0, c->sin[b][0].p, c->sin[b][1].p, len);
    Q.skip_r = 1;
    if ((rc = launch_front<K>(c, hp, Q, true))) return rc;
    CUDA_TRY(c, cudaEventRecord(ev_free[b], e));  // pass 1 consumed buffer b
    if ((rc = launch_pass2<K>(c, hp, Q))) return rc;
    if ((rc = launch_join<K>(c, hp, Q, mat))) return rc;
    if (mat) {
      CUDA_TRY(c, cudaMemcpyAsync(hcur + b, Q.results + RES_CURSOR, 8, cudaMemcpyDeviceToHost, e));
      CUDA_TRY(c, cudaEventRecord(ev_j[b], e));
      if (k >= 1 && (rc = drain(1 - b))) return rc;  // chunk k-1 is done by now or soon
    }
  }
  if (mat && (rc = drain((int)((nch - 1) & 1)))) return rc;
  unsigned long long* h = (unsigned long long*)c->h_res;
  Plan F = device_plan(c, hp, nullptr, nullptr, 0, nullptr, nullptr, 0);
  CUDA_TRY(c, cudaMemcpyAsync(h, F.results, 4 * sizeof(unsigned long long), cudaMemcpyDeviceToHost, e));
  CUDA_TRY(c, cudaEventRecord(ev_d, d));
  CUDA_TRY(c, cudaStreamWaitEvent(e, ev_d, 0));
  CUDA_TRY(c, cudaEventRecord(ev_end, e));
  CUDA_TRY(c, cudaStreamSynchronize(e));
  if (overflow || h[RES_MATCHES] > cap) return join_host_serial(c, Rk, Rp, nR, Sk, Sp, nS, radix_bits, out_mode, res);
  memset(res, 0, sizeof *res);
  res->matches = h[RES_MATCHES];
  res->checksum = h[RES_CHECKSUM];
  res->radix_bits = hp.B;
  res->passes = hp.B >= 2 ? 2 : (hp.B == 1 ? 1 : 0);
  res->kernels = c->launches;
  if (mat) {
    res->r_pay_out = ho;
    res->s_pay_out = ho + cap * pb;
  }
  cudaEventElapsedTime(&res->ms_total, ev_start, ev_end);
  return HJ_OK;
}

int join_host_serial(Ctx* c, const void* Rk, const void* Rp, uint64_t nR, const void* Sk, const void* Sp, uint64_t nS,
                     int radix_bits, int out_mode, hj_result* res) {
  int rc = HJ_OK;
  const size_t kb = c->key_bytes, pb = c->pay_bytes;
  cudaStream_t st = c->stream;
  const void* src[4] = {Rk, Rp, Sk, Sp};
  const size_t bytes[4] = {nR * kb, nR * pb, nS * kb, nS * pb};
  for (int i = 0; i < 4 && rc == HJ_OK; ++i) {
    rc = ensure(c, c->in[i], bytes[i]);
    if (rc == HJ_OK && cudaMemcpyAsync(c->in[i].p, src[i], bytes[i], cudaMemcpyHostToDevice, st) != cudaSuccess)
      rc = fail(c, HJ_ERR_CUDA, "H2D copy failed");
  }
  if (rc == HJ_OK)
    rc = run_join(c, c->in[0].p, c->in[1].p, nR, c->in[2].p, c->in[3].p, nS, radix_bits, out_mode, res);
  if (rc == HJ_OK && out_mode == HJ_OUT_MATERIALIZE && res->matches) {
    const size_t need = 2 * res->matches * pb;
    if (c->h_out_bytes < need) {
      if (c->h_out) cudaFreeHost(c->h_out);
      c->h_out = nullptr;
      c->h_out_bytes = 0;
      if (cudaMallocHost(&c->h_out, need) != cudaSuccess) rc = fail(c, HJ_ERR_OOM, "pinned host alloc of %zu B", need);
      else c->h_out_bytes = need;
    }
    if (rc == HJ_OK) {
      char* ho = (char*)c->h_out;
      if (cudaMemcpyAsync(ho, res->r_pay_out, res->matches * pb, cudaMemcpyDeviceToHost, st) != cudaSuccess ||
          cudaMemcpyAsync(ho + res->matches * pb, res->s_pay_out, res->matches * pb, cudaMemcpyDeviceToHost, st) !=
              cudaSuccess ||
          cudaStreamSynchronize(st) != cudaSuccess)
        rc = fail(c, HJ_ERR_CUDA, "D2H copy of pairs failed");
      res->r_pay_out = ho;
      res->s_pay_out = ho + res->matches * pb;
    }
  }
  return rc;
}

// hj_xd_join's host side: pinned staging, the send plan (c->xd_hp, own metadata buffer), the
// receive plan `hr` (sized by this rank's window capacity capt[] in tuples: the received counts
// are known only on the device), and every device buffer both need. No launches.
int xd_prepare(Ctx* c, int gpu_bits, unsigned long long nR, unsigned long long nS, int local_bits, bool mat,
               const unsigned long long capt[2], HostPlan& hr) {
  const size_t tb = (size_t)c->key_bytes + c->pay_bytes;
  if (!c->xd_hp) {
    c->xd_hp = new HostPlan();
    c->xd_P = new Plan();
  }
  if (!c->h_xd_cur) {
    if (cudaMallocHost(&c->h_xd_cur, (size_t)XD_MAX * 2 * XD_MAX * 8) != cudaSuccess ||
        cudaHostAlloc(&c->h_xd_err, 64, cudaHostAllocMapped) != cudaSuccess ||
        cudaHostGetDevicePointer((void**)&c->d_xd_err, c->h_xd_err, 0) != cudaSuccess)
      return fail(c, HJ_ERR_OOM, "pinned exchange staging");
    *c->h_xd_err = 0;
  }
  HostPlan& hs = *c->xd_hp;
  int rc = prepare(c, hs, nR, nS, local_bits, false, gpu_bits, 1, PLAN_SEND);
  if (rc == HJ_OK) rc = ensure(c, c->xd_meta, hs.meta_bytes);
  if (rc == HJ_OK) rc = ensure(c, c->t1[0], nR * tb + 16);  // overflow scratch for pass 1
  if (rc == HJ_OK) rc = ensure(c, c->t1[1], nS * tb + 16);
  // join capacities from this rank's own row count (its expected share of every relation), not
  // from the window capacity (slack and regrowth inflated C_R: c5_gpu join 3.12 ms at one rank,
  // two join blocks per SM instead of three... against 2.10 on the local path)
  if (rc == HJ_OK) rc = prepare(c, hr, capt[0], capt[1], local_bits, mat, 0, 1 << gpu_bits, PLAN_RECV, nR);
  if (rc == HJ_OK && (hr.npieces() > 1024 || hs.pb() > 10))
    rc = fail(c, HJ_ERR_UNSUPPORTED, "too many pass-1 pieces (G=%d, local_bits=%d)", 1 << gpu_bits, local_bits);
  return rc;
}

}  // namespace

struct hj_ctx {
  Ctx c;
};

extern "C" {

const char* hj_version(void) {
  return "hj-b200 0.1 (sm_100a; nvcc " HJ_STR(__CUDACC_VER_MAJOR__) ")";
}

int hj_create(hj_ctx** out, int device, int key_bytes, int pay_bytes, void* cuda_stream) {
  if (!out) return fail(nullptr, HJ_ERR_INVALID, "out is NULL");
  *out = nullptr;
  if (!((key_bytes == 4 && pay_bytes == 4) || (key_bytes == 8 && pay_bytes == 8)))
    return fail(nullptr, HJ_ERR_UNSUPPORTED, "key/payload widths %d/%d (supported: 4/4, 8/8)", key_bytes, pay_bytes);
  int ndev = 0;
  cudaError_t e = cudaGetDeviceCount(&ndev);
  if (e != cudaSuccess || ndev == 0) return fail(nullptr, HJ_ERR_CUDA, "no CUDA device: %s", cudaGetErrorString(e));
  if (device < 0 || device >= ndev) return fail(nullptr, HJ_ERR_INVALID, "device %d out of range", device);
  hj_ctx* h = new hj_ctx();
  Ctx* c = &h->c;
  c->device = device;
  c->key_bytes = key_bytes;
  c->pay_bytes = pay_bytes;
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(device);
  cudaDeviceProp prop;
  cudaGetDeviceProperties(&prop, device);
  c->num_sms = prop.multiProcessorCount;
  c->smem_optin = prop.sharedMemPerBlockOptin;
  if (prop.major < 10) {
    cudaSetDevice(prev);
    delete h;
    return fail(nullptr, HJ_ERR_UNSUPPORTED, "device %d is sm_%d%d; this library is built for sm_100a", device,
                prop.major, prop.minor);
  }
  int rc = key_bytes == 4 ? set_kernel_attrs<uint32_t>(c) : set_kernel_attrs<uint64_t>(c);
  e = cudaGetLastError();
  if (rc || e != cudaSuccess) {
    cudaSetDevice(prev);
    delete h;
    return fail(nullptr, HJ_ERR_CUDA, "kernel attribute setup failed: %s", cudaGetErrorString(e));
  }
  if (cudaStreamCreateWithFlags(&c->own_stream, cudaStreamNonBlocking) != cudaSuccess ||
      cudaMallocHost(&c->h_res, 8 * 1025 + 64) != cudaSuccess) {
    cudaSetDevice(prev);
    delete h;
    return fail(nullptr, HJ_ERR_CUDA, "stream / pinned allocation failed");
  }
  c->stream = cuda_stream ? (cudaStream_t)cuda_stream : c->own_stream;
  for (auto& ev : c->ev) cudaEventCreate(&ev);
  for (int k = 0; k < 7; ++k) c->ev_own[k] = c->ev[k];
  for (auto& ev : c->sev) cudaEventCreate(&ev);
  cudaStreamCreateWithFlags(&c->h2d_stream, cudaStreamNonBlocking);
  cudaStreamCreateWithFlags(&c->d2h_stream, cudaStreamNonBlocking);
  cudaMallocHost(&c->h_cur, 64);
  cudaSetDevice(prev);
  *out = h;
  return HJ_OK;
}

void hj_destroy(hj_ctx* h) {
  if (!h) return;
  Ctx* c = &h->c;
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  drain_pending(c);  // fills the results of pending hj_join_async calls
  // drain every stream this ctx issued work on before its memory is freed
  for (cudaStream_t s : {c->stream, c->own_stream, c->h2d_stream, c->d2h_stream})
    if (s) cudaStreamSynchronize(s);
  DevBuf* bufs[] = {&c->t1[0], &c->t1[1], &c->t2[0], &c->t2[1], &c->meta,    &c->out_r,    &c->out_s,
                    &c->in[0], &c->in[1], &c->in[2], &c->in[3], &c->xsend[0], &c->xsend[1], &c->xcnt[0],
                    &c->xcnt[1], &c->np_heads, &c->np_next, &c->bc_pool1[0], &c->bc_pool1[1], &c->bc_pool2[0],
                    &c->bc_pool2[1], &c->bc_meta, &c->xd_meta, &c->sin[0][0], &c->sin[0][1], &c->sin[1][0],
                    &c->sin[1][1]};
  for (DevBuf* b : bufs)
    if (b->p && !b->ws) cudaFree(b->p);  // workspace-carved buffers belong to the caller
  if (c->graph) cudaGraphExecDestroy(c->graph);
  for (auto& b : c->xd_win)
    if (b.p) cudaFree(b.p);
  delete c->xd_hp;
  delete c->xd_P;
  if (c->h_xd_cur) cudaFreeHost(c->h_xd_cur);
  if (c->h_xd_err) cudaFreeHost(c->h_xd_err);
  if (c->h_res) cudaFreeHost(c->h_res);
  if (c->h_out) cudaFreeHost(c->h_out);
  for (auto& ev : c->ev)
    if (ev) cudaEventDestroy(ev);
  for (Pending& q : c->pend) {
    for (auto& ev : q.ev)
      if (ev) cudaEventDestroy(ev);
    if (q.h) cudaFreeHost(q.h);
  }
  for (auto& ev : c->sev)
    if (ev) cudaEventDestroy(ev);
  if (c->h_cur) cudaFreeHost(c->h_cur);
  if (c->h2d_stream) cudaStreamDestroy(c->h2d_stream);
  if (c->d2h_stream) cudaStreamDestroy(c->d2h_stream);
  if (c->own_stream) cudaStreamDestroy(c->own_stream);
  cudaSetDevice(prev);
  delete h;
}

const char* hj_last_error(const hj_ctx* h) { return h ? h->c.err.c_str() : g_create_error.c_str(); }

int hj_set_stream(hj_ctx* h, void* s) {
  if (!h) return HJ_ERR_INVALID;
  // NULL is the caller's "stream 0", the legacy default stream (torch's default stream handle is
  // 0): work is then ordered after every kernel the caller issued there (mapping NULL
  // to the ctx's non-blocking stream let the join read columns still being written)
  const cudaStream_t ns = s ? (cudaStream_t)s : cudaStreamLegacy;
  // pending hj_join_async calls use the ctx's buffers on the old stream: finish them before work
  // on another stream could overlap them
  if (ns != h->c.stream)
    if (const int rc_ = drain_pending(&h->c)) return rc_;
  h->c.stream = ns;
  return HJ_OK;
}

int hj_set_option(hj_ctx* h, int opt, int64_t v) {
  if (!h) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  if (v < 0) return fail(c, HJ_ERR_INVALID, "negative option value");
  drop_graph(c);  // any option may change the captured launch sequence: capture again
  switch (opt) {
    case HJ_OPT_CAP_R: c->opt_cap_r = v; break;
    case HJ_OPT_CHUNK_S: c->opt_chunk_s = v; break;
    case HJ_OPT_OUT_CAPACITY: c->opt_out_cap = v; break;
    case HJ_OPT_TIMING: c->opt_timing = v; break;
    case HJ_OPT_BLOCKS_PER_SM: c->opt_bps = v; break;
    case HJ_OPT_STREAM_CHUNK: c->opt_stream_chunk = v; break;
    case HJ_OPT_MAT_CHECKSUM: c->opt_mat_chk = v; break;
    case HJ_OPT_PASS_WS:
      if (v != 0 && v != 1 && v != 18 && v != 20 && v != 22)
        return fail(c, HJ_ERR_INVALID, "pass_ws must be 0 (off), 1 (auto) or 18/20/22 compute warps");
      c->opt_pass_ws = v;
      break;
    case HJ_OPT_PDL: c->opt_pdl = v ? 1 : 0; break;
    case HJ_OPT_PASS_L2PF: c->opt_pass_l2pf = v; break;
    case HJ_OPT_PASS1_BITS: c->opt_pass1_bits = v; break;
    case HJ_OPT_PARTITIONER:
      if (v > 1) return fail(c, HJ_ERR_INVALID, "partitioner must be 0 (histogram) or 1 (bucket chains)");
      c->opt_partitioner = v;
      break;
    case HJ_OPT_GRAPH:
      c->opt_graph = v;
      if (!v && c->graph) {
        cudaGraphExecDestroy(c->graph);
        c->graph = nullptr;
      }
      break;
    case HJ_OPT_JOIN_ALGO:
      if (v > 2) return fail(c, HJ_ERR_INVALID, "join algorithm must be 0, 1 or 2");
      c->opt_join_algo = v;
      break;
    case HJ_OPT_PASS_VARIANT:
      if (v < 0 || v > 4) return fail(c, HJ_ERR_INVALID, "pass variant must be 0..4");
      c->opt_pass_variant = v;
      break;
    case HJ_OPT_PASS_THREADS:
      if (v != 0 && v != 512 && v != 1024) return fail(c, HJ_ERR_INVALID, "pass threads must be 0, 512 or 1024");
      c->opt_pass_nt = v;
      break;
    case HJ_OPT_JOIN_VARIANT:
      if (v > JOIN_NVARIANTS) return fail(c, HJ_ERR_INVALID, "join variant %lld >= %d", (long long)v, JOIN_NVARIANTS);
      c->opt_join_variant = v == 0 ? -1 : v - 1;  // 0 = auto, k = shape k - 1
      break;
    default: return fail(c, HJ_ERR_INVALID, "unknown option %d", opt);
  }
  return HJ_OK;
}

int hj_join(hj_ctx* h, const void* Rk, const void* Rp, uint64_t nR, const void* Sk, const void* Sp, uint64_t nS,
            int radix_bits, int out_mode, hj_result* res) {
  if (!h || !res) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  c->err.clear();
  int rc = check_args(c, Rk, Rp, nR, Sk, Sp, nS, radix_bits, out_mode);
  if (rc) return rc;
  memset(res, 0, sizeof *res);
  if ((rc = drain_pending(c))) return rc;
  if (nR == 0 || nS == 0) return HJ_OK;
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  if (c->ws) {
    ws_begin(c);
    c->use_ws = true;
  }
  rc = run_join(c, Rk, Rp, nR, Sk, Sp, nS, radix_bits, out_mode, res);
  c->use_ws = false;
  cudaSetDevice(prev);
  return rc;
}

int hj_join_async(hj_ctx* h, const void* Rk, const void* Rp, uint64_t nR, const void* Sk, const void* Sp,
                  uint64_t nS, int radix_bits, int out_mode, hj_result* res) {
  if (!h || !res) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  c->err.clear();
  int rc = check_args(c, Rk, Rp, nR, Sk, Sp, nS, radix_bits, out_mode);
  if (rc) return rc;
  memset(res, 0, sizeof *res);
  if (nR == 0 || nS == 0) return HJ_OK;
  // graph replays and the non-partitioned join wait inside the call: run them synchronously
  if (c->opt_graph || c->opt_join_algo == 2) {
    if ((rc = drain_pending(c))) return rc;
    return hj_join(h, Rk, Rp, nR, Sk, Sp, nS, radix_bits, out_mode, res);
  }
  if (c->pend_n == MAX_PENDING && (rc = complete_pending(c))) return rc;
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  Pending& q = c->pend[(c->pend_head + c->pend_n) % MAX_PENDING];
  if (!q.h) {
    for (auto& ev : q.ev)
      if (cudaEventCreate(&ev) != cudaSuccess) ev = nullptr;
    if (cudaMallocHost(&q.h, 16 * sizeof(unsigned long long)) != cudaSuccess) q.h = nullptr;
    if (!q.h || !q.ev[6]) {
      cudaSetDevice(prev);
      return fail(c, HJ_ERR_OOM, "async slot: event / pinned allocation failed");
    }
  }
  q.res = res;
  q.h[5] = 0;
  for (int k = 0; k < 7; ++k) c->ev[k] = q.ev[k];
  c->async = &q;
  if (c->ws) {
    ws_begin(c);
    c->use_ws = true;
  }
  rc = run_join(c, Rk, Rp, nR, Sk, Sp, nS, radix_bits, out_mode, res);
  c->use_ws = false;
  c->async = nullptr;
  for (int k = 0; k < 7; ++k) c->ev[k] = c->ev_own[k];
  if (!rc) c->pend_n++;
  cudaSetDevice(prev);
  return rc;
}

int hj_sync(hj_ctx* h) {
  if (!h) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  const int rc = drain_pending(c);
  cudaSetDevice(prev);
  return rc;
}

uint64_t hj_workspace_bytes(const hj_ctx* hc, uint64_t nR, uint64_t nS, int radix_bits, int out_mode) {
  if (!hc) return 0;
  Ctx* c = const_cast<Ctx*>(&hc->c);
  if (nR == 0 || nS == 0) return 0;
  if (check_args(c, (const void*)1, (const void*)1, nR, (const void*)1, (const void*)1, nS, radix_bits, out_mode))
    return 0;
  hj_result res;
  c->dry = true;
  c->dry_bytes = 0;
  const int rc = run_join(c, nullptr, nullptr, nR, nullptr, nullptr, nS, radix_bits, out_mode, &res);
  c->dry = false;
  return rc ? 0 : (uint64_t)c->dry_bytes;
}

int hj_set_workspace(hj_ctx* h, void* dptr, uint64_t bytes) {
  if (!h) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  c->err.clear();
  if (const int rc_ = drain_pending(c)) return rc_;  // pending hj_join_async calls first
  if (dptr && ((uintptr_t)dptr & 255)) return fail(c, HJ_ERR_INVALID, "workspace must be 256-byte aligned");
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  for (cudaStream_t s : {c->stream, c->own_stream, c->h2d_stream, c->d2h_stream})
    if (s) cudaStreamSynchronize(s);
  // buffers carved from the old workspace are forgotten; hj_join's ctx-owned buffers are freed
  // (everything it needs now comes from the workspace)
  ws_begin(c);
  DevBuf* own[] = {&c->t1[0], &c->t1[1], &c->t2[0], &c->t2[1], &c->meta, &c->out_r, &c->out_s, &c->np_heads,
                   &c->np_next, &c->bc_pool1[0], &c->bc_pool1[1], &c->bc_pool2[0], &c->bc_pool2[1], &c->bc_meta};
  if (dptr)
    for (DevBuf* b : own)
      if (b->p && !b->ws) {
        cudaFree(b->p);
        b->p = nullptr;
        b->bytes = 0;
      }
  drop_graph(c);
  c->ws = (char*)dptr;
  c->ws_bytes = dptr ? (size_t)bytes : 0;
  cudaSetDevice(prev);
  return HJ_OK;
}

int hj_join_host(hj_ctx* h, const void* Rk, const void* Rp, uint64_t nR, const void* Sk, const void* Sp, uint64_t nS,
                 int radix_bits, int out_mode, hj_result* res) {
  if (!h || !res) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  c->err.clear();
  if (const int rc_ = drain_pending(c)) return rc_;  // pending hj_join_async calls first
  int rc = check_args(c, Rk, Rp, nR, Sk, Sp, nS, radix_bits, out_mode);
  if (rc) return rc;
  memset(res, 0, sizeof *res);
  if (nR == 0 || nS == 0) return HJ_OK;
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  // chunk: HJ_OPT_STREAM_CHUNK, else auto (|S| / 16, at least 2^22 tuples; measured on c3)
  const uint64_t chunk = c->opt_stream_chunk > 0 ? (uint64_t)c->opt_stream_chunk
                                                 : std::max<uint64_t>((nS + 15) / 16, 1ull << 22);
  if (chunk >= nS || c->opt_join_algo == 2) rc = join_host_serial(c, Rk, Rp, nR, Sk, Sp, nS, radix_bits, out_mode, res);
  else if (c->key_bytes == 4) rc = join_host_stream<uint32_t>(c, Rk, Rp, nR, Sk, Sp, nS, radix_bits, out_mode, chunk, res);
  else rc = join_host_stream<uint64_t>(c, Rk, Rp, nR, Sk, Sp, nS, radix_bits, out_mode, chunk, res);
  cudaSetDevice(prev);
  return rc;
}

int hj_partition(hj_ctx* h, const void* keys, const void* pays, uint64_t n, int radix_bits, const void** tuples_out,
                 uint64_t* part_start, uint64_t* part_count) {
  if (!h || !tuples_out || !part_start || !part_count) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  c->err.clear();
  if (const int rc_ = drain_pending(c)) return rc_;  // pending hj_join_async calls first
  if (radix_bits < 0 || radix_bits > 20) return fail(c, HJ_ERR_INVALID, "radix_bits must be 0..20");
  if (n && (!keys || !pays)) return fail(c, HJ_ERR_INVALID, "null column with n > 0");
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  HostPlan hp;
  int rc = prepare(c, hp, n, 0, radix_bits, false);
  if (rc == HJ_OK) {
    Plan P = device_plan(c, hp, keys, pays, n, nullptr, nullptr, 0);
    c->launches = 0;
    rc = c->key_bytes == 4 ? launch_front<uint32_t>(c, hp, P) : launch_front<uint64_t>(c, hp, P);
    if (rc == HJ_OK) rc = c->key_bytes == 4 ? launch_pass2<uint32_t>(c, hp, P) : launch_pass2<uint64_t>(c, hp, P);
    if (rc == HJ_OK) {
      const size_t np = (size_t)1 << hp.B;
      unsigned long long* off = new unsigned long long[np + 1];
      cudaError_t e = cudaMemcpyAsync(off, P.rel[0].off, (np + 1) * 8, cudaMemcpyDeviceToHost, c->stream);
      if (e == cudaSuccess) e = cudaStreamSynchronize(c->stream);
      if (e != cudaSuccess) rc = fail(c, HJ_ERR_CUDA, "partition: %s", cudaGetErrorString(e));
      else {
        for (size_t q = 0; q < np; ++q) {
          const size_t d1 = q >> hp.b2, d2 = q & ((1ull << hp.b2) - 1);
          const size_t p = (d2 << hp.b1) | d1;
          part_start[p] = off[q];
          part_count[p] = off[q + 1] - off[q];
        }
        *tuples_out = c->t2[0].p;
      }
      delete[] off;
    }
  }
  cudaSetDevice(prev);
  return rc;
}

int hj_exchange_pack(hj_ctx* h, int rel, const void* keys, const void* pays, uint64_t n, int gpu_bits, int local_bits,
                     const void** send_out, const uint32_t** counts_out, uint64_t* dest_counts) {
  if (!h || !send_out || !counts_out || !dest_counts) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  c->err.clear();
  if (const int rc_ = drain_pending(c)) return rc_;  // pending hj_join_async calls first
  if (rel != 0 && rel != 1) return fail(c, HJ_ERR_INVALID, "rel must be 0 (R) or 1 (S)");
  if (gpu_bits < 0 || gpu_bits > 10 || local_bits < 0 || local_bits > 20)
    return fail(c, HJ_ERR_INVALID, "gpu_bits 0..10, local_bits 0..20");
  if (n && (!keys || !pays)) return fail(c, HJ_ERR_INVALID, "null column with n > 0");
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  HostPlan hp;
  int rc = prepare(c, hp, n, 0, local_bits, false, gpu_bits, 1, PLAN_SEND);
  const size_t tb = (size_t)c->key_bytes + c->pay_bytes;
  const size_t nq = (size_t)1 << hp.qbits();
  if (rc == HJ_OK) rc = ensure(c, c->xsend[rel], n * tb + 16);
  if (rc == HJ_OK) rc = ensure(c, c->xcnt[rel], nq * 4);
  if (rc == HJ_OK) {
    Plan P = device_plan(c, hp, keys, pays, n, nullptr, nullptr, 0);
    P.rel[0].t1 = c->xsend[rel].p;
    P.rel[0].cnt = (uint32_t*)c->xcnt[rel].p;
    c->launches = 0;
    cudaError_t e = cudaMemsetAsync(c->xcnt[rel].p, 0, nq * 4, c->stream);
    if (e != cudaSuccess) rc = fail(c, HJ_ERR_CUDA, "memset: %s", cudaGetErrorString(e));
    if (rc == HJ_OK) rc = c->key_bytes == 4 ? launch_front<uint32_t>(c, hp, P) : launch_front<uint64_t>(c, hp, P);
    if (rc == HJ_OK) {
      const uint32_t F1 = 1u << hp.pb();
      unsigned long long* pst = (unsigned long long*)c->h_res;  // >= F1 + 1 entries (pinned, 8 KB + 64)
      e = cudaMemcpyAsync(pst, P.rel[0].pst, (F1 + 1) * 8, cudaMemcpyDeviceToHost, c->stream);
      if (e == cudaSuccess) e = cudaStreamSynchronize(c->stream);
      if (e != cudaSuccess) rc = fail(c, HJ_ERR_CUDA, "exchange pack: %s", cudaGetErrorString(e));
      else {
        const int G = 1 << gpu_bits;
        for (int j = 0; j < G; ++j) dest_counts[j] = pst[(size_t)(j + 1) << hp.b1] - pst[(size_t)j << hp.b1];
        *send_out = c->xsend[rel].p;
        *counts_out = (const uint32_t*)c->xcnt[rel].p;
      }
    }
  }
  cudaSetDevice(prev);
  return rc;
}

int hj_join_received(hj_ctx* h, const void* R_recv, uint64_t nR, const uint32_t* R_counts, const void* S_recv, uint64_t nS,
                     const uint32_t* S_counts, int nsrc, int local_bits, int out_mode, hj_result* res) {
  if (!h || !res) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  c->err.clear();
  if (const int rc_ = drain_pending(c)) return rc_;  // pending hj_join_async calls first
  if (out_mode != HJ_OUT_COUNT_CHECKSUM && out_mode != HJ_OUT_MATERIALIZE)
    return fail(c, HJ_ERR_INVALID, "bad out_mode %d", out_mode);
  if (nsrc < 1 || nsrc > 1024 || local_bits < 0 || local_bits > 20)
    return fail(c, HJ_ERR_INVALID, "nsrc 1..1024, local_bits 0..20");
  if (!R_counts || !S_counts || (nR && !R_recv) || (nS && !S_recv)) return fail(c, HJ_ERR_INVALID, "null argument");
  memset(res, 0, sizeof *res);
  if (nR == 0 || nS == 0) return HJ_OK;
  const bool mat = out_mode == HJ_OUT_MATERIALIZE;
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  HostPlan hp;
  int rc = prepare(c, hp, nR, nS, local_bits, mat, 0, nsrc, PLAN_RECV);
  if (rc == HJ_OK) {
    Plan P = device_plan(c, hp, nullptr, nullptr, nR, nullptr, nullptr, nS);
    P.rel[0].t1 = const_cast<void*>(R_recv);
    P.rel[1].t1 = const_cast<void*>(S_recv);
    P.prow[0] = R_counts;
    P.prow[1] = S_counts;
    c->launches = 0;
    rc = c->key_bytes == 4 ? launch_front<uint32_t>(c, hp, P) : launch_front<uint64_t>(c, hp, P);
    if (rc == HJ_OK) rc = c->key_bytes == 4 ? launch_pass2<uint32_t>(c, hp, P) : launch_pass2<uint64_t>(c, hp, P);
    if (rc == HJ_OK) rc = finish_join(c, hp, P, mat, res);
  }
  if (rc == HJ_OK && c->h_xd_err && *(volatile uint32_t*)c->h_xd_err) {
    const uint32_t xe = *(volatile uint32_t*)c->h_xd_err;
    *c->h_xd_err = 0;
    rc = fail(c, HJ_ERR_COMM, "exchange barrier timed out: rank %u never reached hj_xd_barrier", xe >> 4);
  }
  cudaSetDevice(prev);
  return rc;
}

// ---- direct-store exchange -----------------------------------------------------------------

int hj_xd_window(hj_ctx* h, int slot, uint64_t bytes, void** dptr, void* ipc_handle, int* grew) {
  if (!h || !dptr) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  c->err.clear();
  if (slot < 0 || slot > 2) return fail(c, HJ_ERR_INVALID, "window slot must be 0 (R), 1 (S) or 2 (flags)");
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  int rc = HJ_OK;
  DevBuf& b = c->xd_win[slot];
  const size_t want = std::max<size_t>(align_up(bytes, 256), 256);
  const bool g = !b.p || b.bytes < want;
  if (g) {
    // plain cudaMalloc (IPC-exportable); peers that mapped the old window must re-open it
    if (b.p) {
      cudaStreamSynchronize(c->stream);
      cudaFree(b.p);
      b.p = nullptr;
      b.bytes = 0;
    }
    cudaError_t e = cudaMalloc(&b.p, want);
    if (e == cudaSuccess) e = cudaMemset(b.p, 0, want);
    if (e != cudaSuccess) {
      b.p = nullptr;
      rc = fail(c, e == cudaErrorMemoryAllocation ? HJ_ERR_OOM : HJ_ERR_CUDA, "window: %s", cudaGetErrorString(e));
    } else {
      b.bytes = want;
    }
  }
  if (rc == HJ_OK) {
    *dptr = b.p;
    if (grew) *grew = g ? 1 : 0;
    if (ipc_handle) {
      cudaIpcMemHandle_t mh;
      cudaError_t e = cudaIpcGetMemHandle(&mh, b.p);
      if (e != cudaSuccess) rc = fail(c, HJ_ERR_CUDA, "cudaIpcGetMemHandle: %s", cudaGetErrorString(e));
      else memcpy(ipc_handle, &mh, sizeof mh);
    }
  }
  cudaSetDevice(prev);
  return rc;
}

uint64_t hj_xd_header_bytes(int G, int local_bits) {
  if (G < 1 || local_bits < 0 || local_bits > 20) return 0;
  return align_up((size_t)G * ((size_t)4 << xchg_b1(G, local_bits)), 256);
}

uint32_t hj_exchange_row_len(int G, int local_bits) {
  if (G < 1 || local_bits < 0 || local_bits > 20) return 0;
  return 1u << xchg_b1(G, local_bits);
}

int hj_ipc_open(hj_ctx* h, const void* ipc_handle, void** dptr) {
  if (!h || !ipc_handle || !dptr) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  c->err.clear();
  static_assert(sizeof(cudaIpcMemHandle_t) == 64, "64-byte IPC handle");
  cudaIpcMemHandle_t mh;
  memcpy(&mh, ipc_handle, sizeof mh);
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  cudaError_t e = cudaIpcOpenMemHandle(dptr, mh, cudaIpcMemLazyEnablePeerAccess);
  cudaSetDevice(prev);
  if (e != cudaSuccess) {
    cudaGetLastError();
    return fail(c, HJ_ERR_CUDA, "cudaIpcOpenMemHandle: %s", cudaGetErrorString(e));
  }
  return HJ_OK;
}

int hj_ipc_close(hj_ctx* h, void* dptr) {
  if (!h || !dptr) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  cudaError_t e = cudaIpcCloseMemHandle(dptr);
  cudaSetDevice(prev);
  if (e != cudaSuccess) return fail(c, HJ_ERR_CUDA, "cudaIpcCloseMemHandle: %s", cudaGetErrorString(e));
  return HJ_OK;
}

int hj_xd_count(hj_ctx* h, const void* Rk, const void* Rp, uint64_t nR, const void* Sk, const void* Sp, uint64_t nS,
                int gpu_bits, int local_bits, uint64_t* dest_counts) {
  if (!h || !dest_counts) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  c->err.clear();
  if (const int rc_ = drain_pending(c)) return rc_;  // pending hj_join_async calls first
  if (gpu_bits < 0 || (1 << gpu_bits) > XD_MAX || local_bits < 0 || local_bits > 20)
    return fail(c, HJ_ERR_INVALID, "gpu_bits 0..6, local_bits 0..20");
  if ((nR && (!Rk || !Rp)) || (nS && (!Sk || !Sp))) return fail(c, HJ_ERR_INVALID, "null column with n > 0");
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  if (!c->xd_hp) {
    c->xd_hp = new HostPlan();
    c->xd_P = new Plan();
  }
  HostPlan& hp = *c->xd_hp;
  int rc = prepare(c, hp, nR, nS, local_bits, false, gpu_bits, 1, PLAN_SEND);
  // the send plan lives in its own buffer: hj_xd_store's pass 1 still reads it (asynchronously)
  // when this rank's hj_join_received prepares its receive plan in c->meta
  if (rc == HJ_OK) rc = ensure(c, c->xd_meta, hp.meta_bytes);
  if (rc == HJ_OK && !c->h_xd_cur) {
    if (cudaMallocHost(&c->h_xd_cur, (size_t)XD_MAX * 2 * XD_MAX * 8) != cudaSuccess ||
        cudaHostAlloc(&c->h_xd_err, 64, cudaHostAllocMapped) != cudaSuccess ||
        cudaHostGetDevicePointer((void**)&c->d_xd_err, c->h_xd_err, 0) != cudaSuccess)
      rc = fail(c, HJ_ERR_OOM, "pinned exchange staging");
    else
      *c->h_xd_err = 0;
  }
  if (rc == HJ_OK) {
    Plan& P = *c->xd_P;
    P = device_plan(c, hp, Rk, Rp, nR, Sk, Sp, nS, c->xd_meta.p);
    c->launches = 0;
    rc = c->key_bytes == 4 ? launch_front<uint32_t>(c, hp, P, false, 1) : launch_front<uint64_t>(c, hp, P, false, 1);
    const uint32_t F1 = 1u << hp.pb();
    unsigned long long* pst = c->h_xd_cur;  // 2 x (F1 + 1) <= 2 x 1025 (staging reused below)
    for (int r = 0; r < 2 && rc == HJ_OK; ++r) {
      cudaError_t e = cudaMemcpyAsync(pst + r * 1025, P.rel[r].pst, (F1 + 1) * 8, cudaMemcpyDeviceToHost, c->stream);
      if (e != cudaSuccess) rc = fail(c, HJ_ERR_CUDA, "xd_count: %s", cudaGetErrorString(e));
    }
    if (rc == HJ_OK) {
      cudaError_t e = cudaStreamSynchronize(c->stream);
      if (e != cudaSuccess) rc = fail(c, HJ_ERR_CUDA, "xd_count: %s", cudaGetErrorString(e));
    }
    if (rc == HJ_OK) {
      const int G = 1 << gpu_bits;
      for (int r = 0; r < 2; ++r) {
        c->xd_pst[r].assign(pst + r * 1025, pst + r * 1025 + F1 + 1);
        for (int j = 0; j < G; ++j)
          dest_counts[r * G + j] = c->xd_pst[r][(size_t)(j + 1) << hp.b1] - c->xd_pst[r][(size_t)j << hp.b1];
      }
    }
  }
  cudaSetDevice(prev);
  return rc;
}

int hj_xd_store(hj_ctx* h, int rank, const uint64_t* totals, void* const* win_R, void* const* win_S) {
  if (!h || !totals || !win_R || !win_S) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  c->err.clear();
  if (const int rc_ = drain_pending(c)) return rc_;  // pending hj_join_async calls first
  if (!c->xd_hp || c->xd_pst[0].empty()) return fail(c, HJ_ERR_INVALID, "hj_xd_store without hj_xd_count");
  HostPlan& hp = *c->xd_hp;
  Plan P = *c->xd_P;
  const int G = 1 << hp.g;
  if (rank < 0 || rank >= G) return fail(c, HJ_ERR_INVALID, "rank %d outside 0..%d", rank, G - 1);
  void* const* win[2] = {win_R, win_S};
  for (int r = 0; r < 2; ++r)
    for (int j = 0; j < G; ++j)
      if (!win[r][j]) return fail(c, HJ_ERR_INVALID, "null window pointer (relation %d, rank %d)", r, j);
  const long long tb = c->key_bytes + c->pay_bytes;
  const size_t H = hj_xd_header_bytes(G, hp.gsh);  // (the send plan's B is its b1; gsh = local bits)
  const uint32_t F1 = 1u << hp.pb();
  // cursor of pass-1 digit D = (j, d1): element offset, from this rank's own window tuples, of
  // where this rank's d1 run for rank j starts in rank j's window (source-major layout, then d1)
  for (int r = 0; r < 2; ++r) {
    const char* base = (const char*)win[r][rank] + H;
    const std::vector<unsigned long long>& pst = c->xd_pst[r];
    for (int j = 0; j < G; ++j) {
      const long long diff = (long long)((const char*)win[r][j] + H - base);
      if (diff % tb) return fail(c, HJ_ERR_INVALID, "window of rank %d not aligned to the tuple size", j);
      unsigned long long seg = 0;
      for (int s = 0; s < rank; ++s) seg += totals[((size_t)r * G + s) * G + j];
      const unsigned long long rel0 = (unsigned long long)(diff / tb) + seg;
      for (uint32_t d1 = 0; d1 < (1u << hp.b1); ++d1) {
        const size_t D = ((size_t)j << hp.b1) | d1;
        c->h_xd_cur[r * 1024 + D] = rel0 + (pst[D] - pst[(size_t)j << hp.b1]);
      }
    }
    P.rel[r].t1 = const_cast<char*>(base);
  }
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  int rc = HJ_OK;
  cudaError_t e = cudaSuccess;
  for (int r = 0; r < 2 && e == cudaSuccess; ++r)
    e = cudaMemcpyAsync(P.rel[r].cur1, c->h_xd_cur + r * 1024, (size_t)F1 * 8, cudaMemcpyHostToDevice, c->stream);
  if (e != cudaSuccess) rc = fail(c, HJ_ERR_CUDA, "xd_store: %s", cudaGetErrorString(e));
  c->launches = 0;
  if (rc == HJ_OK) {
    XdRows a;
    memset(&a, 0, sizeof a);
    a.rowlen = 1u << hp.B;
    for (int r = 0; r < 2; ++r) {
      a.cnt[r] = P.rel[r].cnt;
      for (int j = 0; j < G; ++j) a.dst[r][j] = (uint32_t*)win[r][j] + (size_t)rank * a.rowlen;
    }
    k_xd_rows<<<dim3(G, 2, std::max(1u, std::min(32u, (a.rowlen / 4) / 256))), 256, 0, c->stream>>>(a);
    e = cudaGetLastError();
    if (e != cudaSuccess) rc = fail(c, HJ_ERR_CUDA, "k_xd_rows: %s", cudaGetErrorString(e));
    else c->launches += 1;
  }
  if (rc == HJ_OK)
    rc = c->key_bytes == 4 ? launch_front<uint32_t>(c, hp, P, false, 2) : launch_front<uint64_t>(c, hp, P, false, 2);
  c->xd_pst[0].clear();  // one store per count
  cudaSetDevice(prev);
  return rc;
}

int hj_xd_barrier(hj_ctx* h, int rank, int G, void* const* flags, uint32_t timeout_ms) {
  if (!h || !flags) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  c->err.clear();
  if (G < 1 || G > XD_MAX || rank < 0 || rank >= G) return fail(c, HJ_ERR_INVALID, "G 1..64, 0 <= rank < G");
  if (!c->d_xd_err) return fail(c, HJ_ERR_INVALID, "hj_xd_barrier before hj_xd_count");
  XdBarrier b;
  memset(&b, 0, sizeof b);
  for (int j = 0; j < G; ++j) {
    if (!flags[j]) return fail(c, HJ_ERR_INVALID, "null flag window of rank %d", j);
    b.flags[j] = (unsigned long long*)flags[j];
  }
  b.own = (const unsigned long long*)flags[rank];
  b.epoch = ++c->xd_epoch;
  b.timeout_ns = (unsigned long long)timeout_ms * 1000000ull;
  b.err = c->d_xd_err;
  b.G = G;
  b.rank = rank;
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  k_xd_barrier<<<1, XD_MAX, 0, c->stream>>>(b);
  cudaError_t e = cudaGetLastError();
  cudaSetDevice(prev);
  if (e != cudaSuccess) return fail(c, HJ_ERR_CUDA, "k_xd_barrier: %s", cudaGetErrorString(e));
  return HJ_OK;
}

int hj_xd_reserve(hj_ctx* h, int gpu_bits, uint64_t nR, uint64_t nS, int local_bits, int out_mode, uint64_t win_R_bytes,
                  uint64_t win_S_bytes) {
  if (!h) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  c->err.clear();
  if (gpu_bits < 0 || (1 << gpu_bits) > XD_MAX || local_bits < 0 || local_bits > 20)
    return fail(c, HJ_ERR_INVALID, "gpu_bits 0..6, local_bits 0..20");
  const size_t tb = (size_t)c->key_bytes + c->pay_bytes;
  const size_t H = hj_xd_header_bytes(1 << gpu_bits, local_bits);
  const unsigned long long capt[2] = {win_R_bytes > H + 64 ? (win_R_bytes - H - 64) / tb : 0,
                                      win_S_bytes > H + 64 ? (win_S_bytes - H - 64) / tb : 0};
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  HostPlan hr;
  int rc = xd_prepare(c, gpu_bits, nR, nS, local_bits, out_mode == HJ_OUT_MATERIALIZE, capt, hr);
  cudaSetDevice(prev);
  return rc;
}

int hj_xd_join(hj_ctx* h, int rank, int gpu_bits, const void* Rk, const void* Rp, uint64_t nR, const void* Sk,
               const void* Sp, uint64_t nS, int local_bits, int out_mode, void* const* win_R, void* const* win_S,
               void* const* board, const uint64_t* win_bytes, uint32_t timeout_ms, hj_result* res, uint64_t* totals,
               uint64_t* all) {
  if (!h || !win_R || !win_S || !board || !win_bytes || !res || !totals || !all) return HJ_ERR_INVALID;
  Ctx* c = &h->c;
  c->err.clear();
  if (const int rc_ = drain_pending(c)) return rc_;  // pending hj_join_async calls first
  if (out_mode != HJ_OUT_COUNT_CHECKSUM && out_mode != HJ_OUT_MATERIALIZE)
    return fail(c, HJ_ERR_INVALID, "bad out_mode %d", out_mode);
  if (gpu_bits < 0 || (1 << gpu_bits) > XD_MAX || local_bits < 0 || local_bits > 20)
    return fail(c, HJ_ERR_INVALID, "gpu_bits 0..6, local_bits 0..20");
  const int G = 1 << gpu_bits;
  if (rank < 0 || rank >= G) return fail(c, HJ_ERR_INVALID, "rank %d outside 0..%d", rank, G - 1);
  if ((nR && (!Rk || !Rp)) || (nS && (!Sk || !Sp))) return fail(c, HJ_ERR_INVALID, "null column with n > 0");
  void* const* win[2] = {win_R, win_S};
  for (int j = 0; j < G; ++j)
    if (!win_R[j] || !win_S[j] || !board[j]) return fail(c, HJ_ERR_INVALID, "null window of rank %d", j);
  const bool mat = out_mode == HJ_OUT_MATERIALIZE;
  const size_t tb = (size_t)c->key_bytes + c->pay_bytes;
  const size_t H = hj_xd_header_bytes(G, local_bits);
  XdJoin a;
  memset(&a, 0, sizeof a);
  unsigned long long capt[2];
  for (int r = 0; r < 2; ++r)
    for (int j = 0; j < G; ++j) {
      const uint64_t wb = win_bytes[r * G + j];
      a.cap[r][j] = wb > H + 64 ? (wb - H - 64) / tb : 0;
      const long long diff = (long long)((const char*)win[r][j] - (const char*)win[r][rank]);
      if (diff % (long long)tb) return fail(c, HJ_ERR_INVALID, "window of rank %d not aligned to the tuple size", j);
      a.delta[r][j] = diff / (long long)tb;
      if (j == rank) capt[r] = a.cap[r][j];
    }
  int prev = 0;
  cudaGetDevice(&prev);
  cudaSetDevice(c->device);
  int rc = HJ_OK;
  HostPlan hr;
  if (rc == HJ_OK) rc = xd_prepare(c, gpu_bits, nR, nS, local_bits, mat, capt, hr);
  if (rc != HJ_OK) {
    cudaSetDevice(prev);
    return rc;
  }
  HostPlan& hs = *c->xd_hp;
  Plan Ps = device_plan(c, hs, Rk, Rp, nR, Sk, Sp, nS, c->xd_meta.p);
  Plan Pr = device_plan(c, hr, nullptr, nullptr, capt[0], nullptr, nullptr, capt[1]);
  for (int r = 0; r < 2; ++r) {
    char* own = (char*)win[r][rank];
    Ps.rel[r].t1 = own + H;
    Pr.rel[r].t1 = own + H;
    Pr.prow[r] = (const uint32_t*)own;  // the senders' piece rows; rel[r].cnt: this rank's own histogram
    a.pst[r] = Ps.rel[r].pst;
    a.cur1[r] = Ps.rel[r].cur1;
    a.rows0[r] = (uint32_t*)own;
    a.scratch[r] = ((const char*)c->t1[r].p - (own + H)) / (long long)tb;
    if (((const char*)c->t1[r].p - (own + H)) % (long long)tb)
      rc = fail(c, HJ_ERR_INVALID, "scratch not aligned to the tuple size");
  }
  for (int j = 0; j < G; ++j) a.board[j] = (unsigned long long*)board[j];
  a.own = (const unsigned long long*)board[rank];
  a.res = Pr.results;
  a.sums = Pr.results + 4;
  a.overflow = (uint32_t*)(Pr.results + 6);
  a.err = c->d_xd_err;
  a.epoch = ++c->xd_epoch;
  a.timeout_ns = (unsigned long long)timeout_ms * 1000000ull;
  a.rows_words = (uint32_t)G << xchg_b1(G, local_bits);
  a.G = G;
  a.rank = rank;
  a.b1 = hs.b1;
  cudaStream_t st = c->stream;
  c->launches = 0;
  auto run = [&]() -> int {
    const bool k4 = c->key_bytes == 4;
    mark(c, 0);
    CUDA_TRY(c, cudaMemsetAsync(Ps.counters, 0, hs.zero_bytes, st));
    CUDA_TRY(c, cudaMemsetAsync(Pr.counters, 0, hr.zero_bytes, st));
    {  // a1 over the rank-widened field
      const size_t sm = hs.qbits() <= 15 ? ((size_t)4 << hs.qbits()) : hs.qbits() <= 16 ? ((size_t)2 << hs.qbits()) : 0;
      const void* f = sm ? (k4 ? (const void*)k_hist<uint32_t, true, true> : (const void*)k_hist<uint64_t, true, true>)
                         : (k4 ? (const void*)k_hist<uint32_t, false, false> : (const void*)k_hist<uint64_t, false, false>);
      int g = std::max(2, grid_for(c, f, HIST_NT, sm, (nR + nS + 4095) / 4096 + 2));
      uint32_t gr = (uint32_t)((double)g * (double)nR / (double)std::max<unsigned long long>(nR + nS, 1) + 0.5);
      gr = std::min<uint32_t>(std::max<uint32_t>(gr, 1), (uint32_t)g - 1);
      if (nR == 0) gr = 0;
      if (k4) {
        if (hs.qbits() <= 15) k_hist<uint32_t, true, true, true><<<g, HIST_NT, sm, st>>>(Ps, gr);
        else if (sm) k_hist<uint32_t, true, true, false><<<g, HIST_NT, sm, st>>>(Ps, gr);
        else k_hist<uint32_t, false, true><<<g, HIST_NT, 0, st>>>(Ps, gr);
      } else {
        if (hs.qbits() <= 15) k_hist<uint64_t, true, true, true><<<g, HIST_NT, sm, st>>>(Ps, gr);
        else if (sm) k_hist<uint64_t, true, true, false><<<g, HIST_NT, sm, st>>>(Ps, gr);
        else k_hist<uint64_t, false, true><<<g, HIST_NT, 0, st>>>(Ps, gr);
      }
      CUDA_TRY(c, cudaGetLastError());
      c->launches += 1;
    }
    mark(c, 1);
    if (int e0 = launch_plan(c, hs, Ps)) return e0;
    k_xd_totals<<<1, 256, 0, st>>>(a);
    k_xd_cursors<<<1, 1024, 0, st>>>(a);
    CUDA_TRY(c, cudaGetLastError());
    c->launches += 2;
    // the totals board is final once every rank's phase A arrived (read back with the results)
    CUDA_TRY(c, cudaMemcpyAsync(c->h_xd_cur, (const unsigned long long*)board[rank] + XB_TOT, (size_t)G * 2 * XD_MAX * 8,
                                cudaMemcpyDeviceToHost, st));
    mark(c, 2);
    XdRows xr;
    memset(&xr, 0, sizeof xr);
    xr.rowlen = 1u << hs.B;
    xr.skip = a.overflow;
    for (int r = 0; r < 2; ++r) {
      xr.cnt[r] = Ps.rel[r].cnt;
      for (int j = 0; j < G; ++j) xr.dst[r][j] = (uint32_t*)win[r][j] + (size_t)rank * xr.rowlen;
    }
    k_xd_rows<<<dim3(G, 2, std::max(1u, std::min(32u, (xr.rowlen / 4) / 256))), 256, 0, st>>>(xr);
    CUDA_TRY(c, cudaGetLastError());
    c->launches += 1;
    const bool gd = hs.g > 0;
    int e = hs.tile == 512 * (k4 ? pass_items<uint32_t>() : pass_items<uint64_t>())
                ? (k4 ? (gd ? launch_pass<uint32_t, 1, 512, true>(c, hs, Ps, hs.pb()) : launch_pass<uint32_t, 1, 512, false>(c, hs, Ps, hs.pb()))
                      : (gd ? launch_pass<uint64_t, 1, 512, true>(c, hs, Ps, hs.pb()) : launch_pass<uint64_t, 1, 512, false>(c, hs, Ps, hs.pb())))
                : (k4 ? (gd ? launch_pass<uint32_t, 1, 1024, true>(c, hs, Ps, hs.pb()) : launch_pass<uint32_t, 1, 1024, false>(c, hs, Ps, hs.pb()))
                      : (gd ? launch_pass<uint64_t, 1, 1024, true>(c, hs, Ps, hs.pb()) : launch_pass<uint64_t, 1, 1024, false>(c, hs, Ps, hs.pb())));
    if (e) return e;
    XdBarrier b;
    memset(&b, 0, sizeof b);
    for (int j = 0; j < G; ++j) b.flags[j] = (unsigned long long*)board[j] + XB_FLAGS_B;
    b.own = (const unsigned long long*)board[rank] + XB_FLAGS_B;
    b.epoch = a.epoch;
    b.timeout_ns = a.timeout_ns;
    b.err = a.err;
    b.G = G;
    b.rank = rank;
    k_xd_barrier<<<1, XD_MAX, 0, st>>>(b);
    CUDA_TRY(c, cudaGetLastError());
    c->launches += 1;
    mark(c, 3);
    if (int e1 = k4 ? launch_hist_recv<uint32_t>(c, hr, Pr) : launch_hist_recv<uint64_t>(c, hr, Pr)) return e1;
    if (int e1 = launch_plan(c, hr, Pr)) return e1;
    e = k4 ? launch_pass2<uint32_t>(c, hr, Pr) : launch_pass2<uint64_t>(c, hr, Pr);
    if (e) return e;
    return finish_join(c, hr, Pr, mat, res, &a);
  };
  if (rc == HJ_OK) rc = run();
  if (rc == HJ_OK) {
    const unsigned long long* hh = (const unsigned long long*)c->h_res;
    all[0] = hh[6];
    all[1] = hh[7];
    const bool over = (uint32_t)hh[8] != 0;
    for (int s = 0; s < G; ++s)
        for (int r = 0; r < 2; ++r)
          for (int j = 0; j < G; ++j) totals[((size_t)r * G + s) * G + j] = c->h_xd_cur[((size_t)s * 2 + r) * XD_MAX + j];
    const uint32_t xe = *(volatile uint32_t*)c->h_xd_err;
    if (xe) {
      *c->h_xd_err = 0;
      static const char* phase[] = {"?", "totals (phase A)", "barrier (phase B)", "results (phase C)"};
      rc = fail(c, HJ_ERR_COMM, "exchange timed out at the %s wait: rank %u never arrived", phase[xe & 3], xe >> 4);
    }
    if (rc == HJ_OK && over) {
      rc = HJ_XD_REGROW;
      c->err = "receive windows too small: grow them to the sizes `totals` implies and call again";
    }
  }
  cudaSetDevice(prev);
  return rc;
}

}  // extern "C"
