/*
 * hj.h -- C-ABI of the B200-native radix-partitioned hash join (Sioulas et al., ICDE 2019).
 *
 * The hot path behind this boundary (every step runs in hand-written sm_100a CUDA kernels):
 *   a1 radix histogram of the co-partition id p = key & (2^B - 1)      (north star; the paper
 *      has none)
 *   a2 device-wide exclusive scan -> partition offsets, pass cursors, pass-2 chunk list, join
 *      work list
 *   a3 pass-1 scatter on digit d1 (low ceil(B/2) bits), staged through a shared-memory tile
 *      so HBM writes are contiguous runs (P:265-275 metadata + shuffle space in smem)
 *   a4 pass-2 scatter on digit d2 (next floor(B/2) bits), fixed-size chunks of each pass-1
 *      partition assigned to blocks (bucket-at-a-time analogue)
 *   a5 work planning: oversized co-partitions split into (R chunk x S chunk) items
 *      (P:306-308 long chains decomposed; P:1470-1473 block nested loops)
 *   a6 build a shared-memory chained hash table on the R chunk with atomicExch and 16-bit
 *      offsets (Listing 2)
 *   a7 probe with the S chunk following the chains
 *   a8 aggregate (count + pair checksum) or materialize the (r_pay, s_pay) pairs
 *       with one global atomic per probe round and warp-contiguous stores
 *
 * Result definition (identical for every radix_bits):
 *   J = multiset {(r_pay, s_pay) : r_key == s_key}  (keys compared as unsigned bit patterns,
 *       every value legal, bag semantics for duplicates on both sides)
 *   matches  = |J|
 *   checksum = sum over J of sig(r_pay, s_pay) mod 2^64,
 *              sig(p, q) = fmix64(p ^ (q * 0x9E3779B97F4A7C15)), payloads zero-extended,
 *              fmix64 = splitmix64 finalizer.
 *   The build side is always R as passed (no swap); pairs are (r_pay, s_pay); pair order is
 *   unspecified (compare after sorting).
 *
 * Status codes: every int-returning entry point returns HJ_OK or a negative HJ_ERR_*;
 * hj_last_error() gives the message of the last failure on that context.
 */
#ifndef HJ_H_
#define HJ_H_

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef struct hj_ctx hj_ctx; /* opaque; not thread-safe; use one per stream / thread */

enum hj_out_mode {
  HJ_OUT_COUNT_CHECKSUM = 0, /* matches + checksum only (the paper's aggregation) */
  HJ_OUT_MATERIALIZE = 1     /* also the pairs, SoA r_pay_out[] / s_pay_out[]   */
};

enum hj_status {
  HJ_OK = 0,
  HJ_ERR_INVALID = -1,     /* bad argument (null pointer with n > 0, bad mode, bad width ...) */
  HJ_ERR_UNSUPPORTED = -2, /* key/payload widths other than 4/4 and 8/8; radix_bits > 20     */
  HJ_ERR_OOM = -3,         /* device or pinned-host allocation failed                         */
  HJ_ERR_CUDA = -4,        /* any CUDA runtime error; message in hj_last_error()              */
  HJ_ERR_COMM = -5,        /* multi-GPU exchange: a peer missed the hj_xd_barrier deadline    */
  HJ_ERR_WORKSPACE = -6    /* hj_join with a caller workspace (hj_set_workspace): the workspace
                              is smaller than hj_workspace_bytes() for this call, or the
                              materialized pairs outgrew HJ_OPT_OUT_CAPACITY -- then res->matches
                              holds the exact count; raise the capacity, resize, call again      */
};

enum hj_option {
  HJ_OPT_CAP_R = 1,        /* max R tuples per join item (shared-memory build capacity C_R);
                              0 = auto (1.25x the mean R partition, >= 512)                  */
  HJ_OPT_CHUNK_S = 2,      /* max S tuples per join item (C_S); 0 = auto                      */
  HJ_OPT_OUT_CAPACITY = 3, /* initial materialization capacity in pairs; 0 = max(nS, 1M)      */
  HJ_OPT_TIMING = 4,       /* 1 = record per-phase CUDA events into hj_result (default 1)     */
  HJ_OPT_BLOCKS_PER_SM = 5, /* persistent-grid residency override for the passes (0 = auto)   */
  HJ_OPT_JOIN_VARIANT = 6,  /* join kernel shape (tuning; 0 = auto, k = shape k-1 of hj_api.cu's
                               JOIN_SHAPES, 1..9)                                                */
  HJ_OPT_PASS_THREADS = 7,  /* partition-pass block size 512 / 1024 (0 = auto)                   */
  HJ_OPT_JOIN_ALGO = 9,     /* 0 = radix-partitioned + smem hash table (default); 1 = radix-
                               partitioned + ballot nested loops (Listing 1); 2 = non-
                               partitioned hash join on a device-memory table (Fig. 8) */
  HJ_OPT_GRAPH = 11,        /* 1 = hj_join captures its launch sequence in a CUDA graph and replays
                               it while the call signature is unchanged (launch gaps and host
                               preparation leave the critical path: c3 2.73 -> 2.68 ms/call; only
                               ms_total is reported in this mode). Any hj_set_option call drops
                               the captured graph                                                */
  HJ_OPT_PARTITIONER = 12,  /* hj_join only: 0 = histogram + prefix sum + exact placement (north
                               star, default); 1 = the paper's histogram-free bucket chains
                               (NEXT-1): no histogram pass, partitions are chains of
                               buckets from a pool, pass 2 takes one bucket at a time; a pass-2
                               partition that keeps closing buckets takes growing regions of
                               1, 1, 2, 4, 8, 16 consecutive buckets (skew). Needs more device
                               memory (bucket slack: pass-2 pool <= (2n / cap + 2^B + 1) buckets
                               of cap + tile tuples per relation); ms_kernel[0..1] are 0 and
                               ms_kernel[2..3] include each pass's bucket bookkeeping. Ignored by
                               hj_join_host / hj_partition / the exchange calls and by graph mode */
  HJ_OPT_PASS_L2PF = 17,    /* partition passes: 1 = TMA-prefetch each block's unit-after-next into L2
                               (cp.async.bulk.prefetch.L2) when its descriptor is published; 0 = off;
                               2 = auto (default: on for 8-byte keys, where it was measured faster) */
  HJ_OPT_PASS1_BITS = 18,   /* radix bits of pass 1 (0 = auto = ceil(B/2)); pass 2 takes the rest.
                               Each pass's fan-out must stay <= 2^10                              */
  HJ_OPT_PASS_VARIANT = 19, /* partition passes with 1024-thread tiles: either 1024 threads with the
                               next tile prefetched into registers, or the same tile as 512 threads
                               x twice the tuples, no register prefetch, two blocks per SM. Value =
                               1 + mask of the passes using the second form (bit 0 pass 1, bit 1
                               pass 2); 0 = auto (pass 1 of 8-byte tuples, where it measured faster) */
  HJ_OPT_STREAM_CHUNK = 8,  /* hj_join_host: S tuples per streamed chunk (0 = auto = |S|/16, at
                               least 2^22; >= |S| = copy everything, then join)                   */
  HJ_OPT_PASS_WS = 21,      /* partition passes (histogram partitioner, fan-out <= 2^9): 1 (default) =
                               warp-specialized pipeline (a producer warp feeding three TMA stages,
                               compute warps that rank and shuffle each stage in place, writer warps
                               that stream the previous stage out), 20 compute warps (18 for 8-byte
                               tuples on the histogram partitioner); 18/20/22 =
                               that many compute warps (tuning); 0 = every warp of the block in lock
                               step (round-1 kernel)                                                */
  HJ_OPT_PDL = 22,          /* 1 = the planner, the passes and the join are launched with programmatic
                               dependent launch (each starts while its predecessor's last blocks
                               run and waits in-kernel for its results); 0 (default) = plain
                               stream order                                                         */
  HJ_OPT_MAT_CHECKSUM = 20  /* 1 (default) = MATERIALIZE also fills res->checksum (the pairs'
                               signatures are summed by the probe, so every materialized result is
                               self-checking); 0 = checksum left 0 in MATERIALIZE (measurement)   */
};

typedef struct hj_result {
  uint64_t matches;      /* |R ⋈ S| (always filled)                                              */
  uint64_t checksum;     /* sum of sig(r_pay, s_pay) mod 2^64 over the matched pairs, in both
                            modes (MATERIALIZE: unless HJ_OPT_MAT_CHECKSUM = 0)                  */
  const void* r_pay_out; /* MATERIALIZE: `matches` payloads of R, pay_bytes each (device memory
                            for hj_join, pinned host memory for hj_join_host); owned by the ctx,
                            valid until the next join on this ctx or hj_destroy                   */
  const void* s_pay_out; /* same, payloads of S                                                  */
  uint64_t n_items;      /* join work items executed (co-partition x R chunk x S chunk)          */
  int radix_bits;        /* B actually used                                                      */
  int passes;            /* partitioning passes (2 for B >= 2)                                   */
  float ms_total;        /* CUDA-event time of the whole call (first kernel -> result ready)     */
  float ms_partition;    /* histogram + scan + both passes                                      */
  float ms_join;         /* build + probe + output                                              */
  float ms_kernel[5];    /* per step, CUDA events on the ctx stream: 0 histogram, 1 planner,
                            2 pass 1, 3 pass 2, 4 join (HJ_OPT_TIMING = 1)                       */
  uint32_t kernels;      /* kernels this call launched                                           */
  uint32_t reserved;
} hj_result;

/* Create a context on CUDA device `device` for key/payload widths 4/4 or 8/8 bytes.
 * cuda_stream: a cudaStream_t to issue all work on (NULL = a ctx-owned non-blocking stream; the
 * caller then orders it after its own producers, or re-targets it with hj_set_stream).
 * Returns HJ_OK and *out, or HJ_ERR_INVALID / HJ_ERR_UNSUPPORTED / HJ_ERR_CUDA. */
int hj_create(hj_ctx** out, int device, int key_bytes, int pay_bytes, void* cuda_stream);

/* Free every ctx-owned device and host allocation. NULL-safe. */
void hj_destroy(hj_ctx* ctx);

/* Message of the last failure on ctx ("" if none). NULL ctx -> message of the last hj_create. */
const char* hj_last_error(const hj_ctx* ctx);

/* Re-target the context to another stream. NULL = the legacy default stream ("stream 0", e.g.
 * torch's default stream): the join is then ordered after every kernel the caller issued there.
 * Every call is stream-ordered after prior work on the ctx's stream; inputs produced on another
 * stream must be synchronized by the caller. */
int hj_set_stream(hj_ctx* ctx, void* cuda_stream);

/* Set a tuning / test knob (enum hj_option). Results never depend on knobs. */
int hj_set_option(hj_ctx* ctx, int option, int64_t value);

/* R ⋈ S on GPU-resident columns. All four column pointers are DEVICE pointers on ctx's device,
 * caller-owned, read-only, 16-byte alignment recommended (else a scalar-load path is used),
 * and must stay valid until the call returns. Widths are those given to hj_create.
 *   radix_bits: B < 0 = auto (mean R partition ~4096 tuples), 0 = one co-partition (pure
 *               block-nested-loop smem join), 1..20 = 2^B co-partitions in two passes.
 *   out_mode:   enum hj_out_mode.
 * Synchronous: returns once *res is valid (matches/checksum copied to the host, pairs in HBM).
 * nR == 0 or nS == 0 -> HJ_OK with zero results. */
int hj_join(hj_ctx* ctx,
            const void* R_keys, const void* R_pay, uint64_t nR,
            const void* S_keys, const void* S_pay, uint64_t nS,
            int radix_bits, int out_mode, hj_result* res);

/* Asynchronous hj_join: the same work, enqueued on ctx's stream; returns once it is enqueued
 * (host preparation of the next call overlaps this one's kernels: queued back to back, the
 * kernels of consecutive joins leave no host round trip between them). *res is caller-owned and
 * is filled by hj_sync (or by any later call on ctx that completes it); the column pointers must
 * stay valid until then. At most HJ_MAX_PENDING calls are pending per ctx: one more first
 * completes the oldest. Every other call on ctx that touches its buffers (hj_join, hj_join_host,
 * hj_partition, the exchange calls, hj_set_workspace, hj_set_stream to another stream, hj_destroy)
 * first completes all pending calls and fails with the first of their errors, if any.
 * MATERIALIZE: pending calls share the ctx's output buffer, so once hj_sync returns it holds the
 * pairs of the LAST call; a call whose pairs outgrew HJ_OPT_OUT_CAPACITY is not re-run -- its
 * completion fails with HJ_ERR_WORKSPACE and res->matches = the exact count. Graph mode
 * (HJ_OPT_GRAPH) and HJ_OPT_JOIN_ALGO = 2 run synchronously (res filled on return). */
#define HJ_MAX_PENDING 8
int hj_join_async(hj_ctx* ctx,
                  const void* R_keys, const void* R_pay, uint64_t nR,
                  const void* S_keys, const void* S_pay, uint64_t nS,
                  int radix_bits, int out_mode, hj_result* res);

/* Complete every pending hj_join_async call of ctx, in issue order (each one's *res filled).
 * Returns HJ_OK or the first failure among them (hj_last_error: its message). */
int hj_sync(hj_ctx* ctx);

/* Caller-provided device workspace (device buffers reserved up front).
 * hj_workspace_bytes: the device bytes hj_join(ctx, nR, nS, radix_bits, out_mode) needs with the
 *   ctx's current options (partitioner, join algorithm, HJ_OPT_OUT_CAPACITY); 0 if nR or nS is 0
 *   or an argument is invalid. Host-only, no device work.
 * hj_set_workspace: from now on hj_join carves every device buffer from [dptr, dptr + bytes)
 *   (256-byte aligned; e.g. a torch tensor) instead of allocating: no cudaMalloc and no
 *   synchronization inside hj_join before its final result readback. The buffer is caller-owned
 *   and must stay valid (and unused by the caller) while the ctx may use it; materialized pairs
 *   are returned inside it. dptr = NULL returns to ctx-owned allocations. Synchronizes the ctx's
 *   streams and frees hj_join's ctx-owned buffers. hj_join_host / hj_partition / the exchange
 *   calls keep ctx-owned allocations. A too-small workspace -> HJ_ERR_WORKSPACE. */
uint64_t hj_workspace_bytes(const hj_ctx* ctx, uint64_t nR, uint64_t nS, int radix_bits, int out_mode);
int hj_set_workspace(hj_ctx* ctx, void* dptr, uint64_t bytes);

/* Same join from HOST columns (pinned for full overlap; pageable works): the streaming probe
 * of the paper's out-of-GPU strategy (NEXT-3). R is copied and
 * partitioned once; S is copied in chunks (HJ_OPT_STREAM_CHUNK) on a copy stream into two
 * device buffers while the compute stream partitions and joins the previous chunk with the
 * resident R; MATERIALIZE pairs are drained to ctx-owned pinned host memory on a third stream
 * as chunks finish (res->r_pay_out / s_pay_out, valid until the next call on ctx). If the result
 * outgrows the device output buffer the call redoes the join with everything copied first. */
int hj_join_host(hj_ctx* ctx,
                 const void* R_keys, const void* R_pay, uint64_t nR,
                 const void* S_keys, const void* S_pay, uint64_t nS,
                 int radix_bits, int out_mode, hj_result* res);

/* Steps a1-a4 alone on one relation (for parity tests and the multi-GPU exchange): radix
 * partition n device tuples into 2^B co-partitions with the same two passes hj_join uses.
 * Outputs (ctx-owned, valid until the next call on ctx):
 *   *tuples_out: device pointer to n AoS tuples (4/4: uint64 = key | pay << 32;
 *                8/8: {uint64 key; uint64 pay}), co-partition p stored contiguously at
 *                [part_start[p], part_start[p] + part_count[p]), order inside a partition
 *                unspecified.
 *   part_start, part_count: HOST arrays of 2^B entries (caller-allocated), indexed by
 *                p = key & (2^B - 1).
 * B must be 0..20. */
int hj_partition(hj_ctx* ctx, const void* keys, const void* pays, uint64_t n, int radix_bits,
                 const void** tuples_out, uint64_t* part_start, uint64_t* part_count);

/* ---- multi-GPU exchange; the caller runs the collectives in between ------
 * Co-partitions are independent, so G = 2^gpu_bits ranks each own the co-partitions
 * whose radix field is extended by gpu_bits on top: rank j = (key >> local_bits) & (G - 1).
 * The local field splits into b1 = min(ceil(local_bits / 2), 10 - gpu_bits) pass-1 bits and
 * local_bits - b1 pass-2 bits (<= 10), the same on sender and receiver.
 *
 * Count rows: a sender counts only its pass-1 pieces, (destination rank, d1) = 2^(gpu_bits + b1)
 * <= 2^10 shared-memory bins, whatever local_bits is; row j (2^b1 uint32, hj_exchange_row_len)
 * = the tuples of each pass-1 digit d1 sent to rank j. A receiver counts its own 2^local_bits
 * co-partitions of what it received (after the exchange the keys are dense per bin; c5 at G = 8
 * would otherwise need 2^19 sender bins in global memory) and checks the rows against it.
 *
 * hj_exchange_pack: rows a1-a3 on this rank's `n` SoA tuples of relation `rel` (0 = R, 1 = S),
 * with the pass-1 digit widened by the rank bits, so the send buffer is grouped by destination
 * rank and, inside each rank's segment, by the local pass-1 digit d1.
 *   *send_out:   device, n AoS tuples (layout as hj_partition), ctx-owned until the next pack of
 *                the same rel; rank j's segment starts at sum_{i<j} dest_counts[i].
 *   *counts_out: device, [G][2^b1] uint32 piece counts (row j goes to rank j). ctx-owned.
 *   dest_counts: HOST array of G uint64 (caller-allocated): tuples destined to each rank. */
int hj_exchange_pack(hj_ctx* ctx, int rel, const void* keys, const void* pays, uint64_t n, int gpu_bits,
                     int local_bits, const void** send_out, const uint32_t** counts_out, uint64_t* dest_counts);

/* hj_join_received: rows a4-a8 on what this rank received: R_recv / S_recv are device AoS tuples
 * concatenated in source-rank order (each source's segment grouped by d1, as packed), and
 * R_counts / S_counts are device [nsrc][2^b1] uint32 piece-count rows (row s = what source s sent,
 * i.e. source s's counts_out row for this rank). The rank histograms its own 2^local_bits
 * co-partitions of the first sum(rows) received tuples; rows that do not match what the buffers
 * hold (per pass-1 digit), or describe more than nR / nS tuples, fail with HJ_ERR_INVALID and
 * nothing is written. Results are this rank's share of the join (sum matches / checksums over
 * ranks mod 2^64; the union of the materialized pairs). */
int hj_join_received(hj_ctx* ctx, const void* R_recv, uint64_t nR, const uint32_t* R_counts,
                     const void* S_recv, uint64_t nS, const uint32_t* S_counts, int nsrc, int local_bits,
                     int out_mode, hj_result* res);

/* ---- Direct-store exchange (multi-GPU over NVLink / NVSwitch peer memory) -----------------
 * The B200-native form of SURVEY.md §8(e): instead of pack -> NCCL all-to-all -> receive, pass 1
 * of every sender stores each tuple straight into the receive window of the rank that owns its
 * co-partition (peer stores over NVLink; the WC-staged runs arrive as full lines), so the
 * exchange is fused into the partitioning pass and the 2w B/tuple staging round trip and the
 * separate collective disappear. Co-partitions are independent, so rank j owns the
 * co-partitions with (key >> local_bits) & (G - 1) == j, exactly as for hj_exchange_pack.
 *
 * Protocol per join (G = 2^gpu_bits ranks, one context per rank, all calls on ctx's stream):
 *   1. hj_xd_count     rows a1-a2 for R and S: histogram over (rank bits, local bits) + plan;
 *                      returns the tuples this rank sends to every rank.
 *   2. (caller)        all-gather of those [2][G] totals -> totals[2][G][G] on every rank;
 *                      grow windows if needed (hj_xd_window) and exchange their IPC handles.
 *   3. hj_xd_store     row a3: pass 1 writing into the peers' windows, plus this rank's count
 *                      rows into every peer's window header.
 *   4. hj_xd_barrier   every rank's stores are visible before any rank reads its window.
 *   5. hj_join_received(window_R + H, nR_in, window_R, window_S + H, nS_in, window_S, G, ...)
 *                      rows a4-a8 on what arrived (H = hj_xd_header_bytes(G, local_bits)).
 *
 * Receive window of relation r on rank j (ctx-owned device allocation, exported by IPC):
 *   [0, H)      piece-count rows, [G][2^b1] uint32, row s = what source s sent per pass-1 digit
 *               (as hj_exchange_pack's counts_out rows)
 *   [H, ...)    tuples (AoS as hj_partition), source-major: source s's segment starts at
 *               sum_{s' < s} totals[r][s'][j] tuples and is grouped by the local pass-1 digit.
 * Board window (slot 2, HJ_XD_BOARD_BYTES): starts with uint64[HJ_XD_MAX_RANKS] barrier flags,
 * flag s = last barrier epoch source s reached (the rest serves hj_xd_join).
 * Requires G <= HJ_XD_MAX_RANKS; the pass split is hj_exchange_pack's (b1 = min(ceil(local_bits
 * / 2), 10 - gpu_bits)). */
#define HJ_XD_MAX_RANKS 64
/* Board window (slot 2) bytes: barrier / phase flags, the totals board [src][2][dst] and the
 * results board [src][2] of hj_xd_join, all uint64. */
#define HJ_XD_BOARD_BYTES 69632
/* hj_xd_join return value (not an error): some rank's receive window is too small for this
 * call; nothing was joined; grow every window to the size `totals` implies and call again. */
#define HJ_XD_REGROW 1

/* hj_xd_window: (re)allocate ctx's window `slot` (0 = R receive, 1 = S receive, 2 = board) to
 * at least `bytes` (zero-filled when (re)allocated; kept when already large enough).
 *   *dptr:       device pointer of the window in this process (ctx-owned until hj_destroy or
 *                the next growth of the same slot).
 *   ipc_handle:  if non-NULL, 64 bytes receiving cudaIpcGetMemHandle of the window.
 *   *grew:       if non-NULL, 1 when the window was (re)allocated (peers must re-open it). */
int hj_xd_window(hj_ctx* ctx, int slot, uint64_t bytes, void** dptr, void* ipc_handle, int* grew);

/* Bytes of a receive window's count-row header: round_up(G * hj_exchange_row_len * 4, 256). */
uint64_t hj_xd_header_bytes(int G, int local_bits);

/* Entries of one exchange count row: 2^b1, b1 = min(ceil(local_bits / 2), 10 - log2 G). 0 for
 * invalid arguments. */
uint32_t hj_exchange_row_len(int G, int local_bits);

/* hj_ipc_open: map a peer's window (64-byte handle from its hj_xd_window) into this process on
 * ctx's device (cudaIpcMemLazyEnablePeerAccess); hj_ipc_close unmaps it. A handle exported by
 * this same process cannot be opened here (CUDA IPC rule): use the window pointer directly. */
int hj_ipc_open(hj_ctx* ctx, const void* ipc_handle, void** dptr);
int hj_ipc_close(hj_ctx* ctx, void* dptr);

/* hj_xd_count: rows a1-a2 on this rank's SoA rows of R (nR) and S (nS) with the radix field
 * widened by gpu_bits rank bits above local_bits. Synchronous. The plan is kept in ctx for the
 * next hj_xd_store. dest_counts: HOST uint64[2][G] (caller-allocated), dest_counts[r*G + j] =
 * tuples of relation r this rank sends to rank j. Columns must stay unchanged until hj_xd_store. */
int hj_xd_count(hj_ctx* ctx, const void* R_keys, const void* R_pay, uint64_t nR, const void* S_keys,
                const void* S_pay, uint64_t nS, int gpu_bits, int local_bits, uint64_t* dest_counts);

/* hj_xd_store: row a3 of the last hj_xd_count, writing into the peers' receive windows.
 *   rank:       this rank, 0 <= rank < G.
 *   totals:     HOST uint64[2][G][G], totals[(r*G + s)*G + j] = tuples of relation r rank s
 *               sends to rank j (the all-gathered dest_counts of every rank).
 *   win_R/win_S: HOST arrays of G device pointers, valid in this process: every rank's R / S
 *               receive window (this rank's own window at [rank]); each at least
 *               H + (sum_s totals[r][s][j]) * (key_bytes + pay_bytes) bytes.
 * Asynchronous on ctx's stream. */
int hj_xd_store(hj_ctx* ctx, int rank, const uint64_t* totals, void* const* win_R, void* const* win_S);

/* hj_xd_barrier: on ctx's stream, a one-block kernel publishes this rank's epoch to flag
 * [rank] of every rank's flag window (system-scope release after a system fence) and waits
 * until its own flag window holds the epoch of every rank (acquire). The epoch is a per-ctx
 * counter: all ranks must call it the same number of times. flags: HOST array of G device
 * pointers (every rank's flag window, this rank's at [rank]). A rank that waits longer than
 * timeout_ms gives up; the next hj_join_received on ctx then fails with HJ_ERR_COMM.
 * Asynchronous. */
int hj_xd_barrier(hj_ctx* ctx, int rank, int G, void* const* flags, uint32_t timeout_ms);

/* hj_xd_join: the whole multi-GPU join of this rank, driven from the device -- no host round
 * trip and no host collective between the histogram and the result (steps 1-5 above, with the
 * totals exchange and the result reduction done through the peers' boards):
 *   a1-a2 histogram + plan over the rank-widened field; phase A: this rank's [2][G] destination
 *   totals stored into every rank's board, flag A; wait for all flags A; pass-1 cursors from the
 *   board (window capacities checked on the device, identically on every rank); count rows to
 *   the peers' window headers; a3 pass 1 storing into the peers' windows; phase B barrier; a4-a8
 *   on this rank's window; phase C: (matches, checksum) into every board, flag C, wait, sum.
 *   rank, gpu_bits:   this rank, G = 2^gpu_bits ranks (G <= HJ_XD_MAX_RANKS).
 *   columns:          this rank's SoA rows of R and S (device, as hj_join).
 *   win_R, win_S, board: HOST arrays of G device pointers valid in this process (this rank's own
 *                     windows at [rank]; the board of HJ_XD_BOARD_BYTES, zeroed at creation).
 *   win_bytes:        HOST uint64[2][G], the byte size of every rank's R / S window.
 *   res:              this rank's share (as hj_join_received; materialized pairs stay local).
 *   totals:           HOST out uint64[2][G][G], totals[(r*G + s)*G + j] = tuples of relation r
 *                     rank s sent to rank j.
 *   all:              HOST out uint64[2]: matches and checksum summed over all ranks (mod 2^64).
 * Returns HJ_OK, HJ_XD_REGROW (every rank returns it in the same call), or an error;
 * HJ_ERR_COMM when a phase wait exceeded timeout_ms. Synchronous. */
int hj_xd_join(hj_ctx* ctx, int rank, int gpu_bits, const void* R_keys, const void* R_pay, uint64_t nR,
               const void* S_keys, const void* S_pay, uint64_t nS, int local_bits, int out_mode, void* const* win_R,
               void* const* win_S, void* const* board, const uint64_t* win_bytes, uint32_t timeout_ms,
               hj_result* res, uint64_t* totals, uint64_t* all);

/* hj_xd_reserve: every allocation the hj_xd_join call with these sizes (and this rank's window
 * sizes) would make, without launching anything. hj_xd_join synchronizes only at its end, but a
 * first-time device allocation inside it can synchronize the device; ranks that share one GPU
 * (tests) reserve first so no allocation runs while a peer's kernels wait on this rank. */
int hj_xd_reserve(hj_ctx* ctx, int gpu_bits, uint64_t nR, uint64_t nS, int local_bits, int out_mode,
                  uint64_t win_R_bytes, uint64_t win_S_bytes);

/* Library build string (compile flags, arch). */
const char* hj_version(void);

#ifdef __cplusplus
}
#endif

#endif /* HJ_H_ */
