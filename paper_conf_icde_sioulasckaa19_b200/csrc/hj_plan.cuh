// hj_plan.cuh -- device-side plan shared by all kernels of one hj_join call.
#pragma once
#include <cstdint>

#include "hj_common.cuh"

namespace hj {

// Radix field and co-partition order. The local radix field p = key & (2^B - 1) splits into
// d1 = p & (2^b1 - 1) (pass 1) and d2 = p >> b1 (pass 2). Counts, offsets and cursors use q-order
// q = d1 << b2 | d2, so pass-1 partition d1 is the contiguous q range [d1 << b2, (d1 + 1) << b2).
// Multi-GPU exchange: the sender only needs its pass-1 layout, so its plan has
// B = b1, b2 = 0 and the pass-1 digit widened by g rank bits taken from just above the LOCAL field:
//   D = ((key >> gsh) & (2^g - 1)) << b1 | d1        (pb = g + b1 <= 10 bits, gsh = local bits)
// -- a histogram of <= 2^10 bins whatever the local field (c5 at G = 8: 3 + 7 bits, not 3 + 16).
// The receiver counts the 2^B co-partitions of what it received itself (k_hist_recv: keys are
// dense per bin only after the exchange) and takes the pieces' sizes from the senders' rows.
// Pass 2 reads "pieces": piece i = (source s, D) = (i >> pb, i & (2^pb - 1)); on one GPU the
// pieces are the pass-1 partitions, on the exchange receiver the d1-segments sent by each rank.
enum { PLAN_FULL = 0, PLAN_SEND = 1, PLAN_RECV = 2 };

struct RelDev {
  const void* keys;  // SoA input (caller-owned)
  const void* pays;
  unsigned long long n;
  void* t1;                   // pass-1 output / pass-2 input, AoS (the receive buffer on PLAN_RECV)
  void* t2;                   // pass-2 output, AoS, co-partitions contiguous in q-order
  uint32_t* cnt;              // nsrc rows of [2^qbits] counts, q-order (k_hist writes row 0)
  unsigned long long* off;    // [2^qbits + 1] co-partition start (counts summed over rows)
  unsigned long long* cur1;   // [2^pb] pass-1 reservation cursors
  unsigned long long* cur2;   // [2^qbits] pass-2 reservation cursors
  unsigned long long* pst;    // [npieces + 1] pass-2 input piece starts in t1
  uint32_t* cst;              // [npieces + 1] pass-2 chunk prefix (chunks of C2 tuples per piece)
  uint32_t* hot;              // [1 + 2^pb] skew hints from the histogram (k_plan; HOT_NONE = none):
                              // [0] the pass-1 digit holding > 1/4 of the relation, [1 + D] the
                              // d2 digit holding > 1/4 of pass-1 partition D (pass 2)
};
constexpr uint32_t HOT_NONE = 0xffffffffu;

// NEXT-1: the paper's histogram-free partitioner (§III-A). Each pass writes,
// per output partition, a chain of fixed-capacity buckets taken from a pool with atomics; no
// histogram is read and partitions are not contiguous (see hj_bucket.cuh).
struct BcRel {
  void* pool1;                // pass-1 buckets: bucket b holds tuples [b * bsz1, b * bsz1 + fill1[b])
  void* pool2;                // pass-2 buckets
  unsigned long long* st1;    // [2^b1] pass-1 partition state: j << 32 | fill, current bucket =
                              //        p (j = 0, the partition's initial bucket) or np + j - 1
  unsigned long long* st2;    // [2^B]  pass-2 partition state (index q = D << b2 | d2); its high
                              //        word is j | lgk << BC_LGK_SHIFT (region of 2^lgk buckets)
  uint32_t* fill1;            // [nbmax1] tuples in each pass-1 bucket
  uint32_t* part1;            // [nbmax1] pass-1 partition D of each overflow bucket (b >= np1)
  uint32_t* fill2;            // [nbmax2]
  uint32_t* part2;            // [nbmax2] co-partition q of each bucket
  uint4* sl;                  // join slices {offset lo, offset hi, tuples, 0}, grouped by q
  uint32_t* nsl;              // [2^B] join slices of each co-partition's closed buckets
  uint32_t* sst;              // [2^B + 1] first slice of each co-partition
  uint32_t* scur;             // [2^B] slice scatter cursors
  uint32_t np1, np2;          // partitions per pass (2^b1, 2^B): buckets [0, np) are the initial ones
  uint32_t cap1, cap2;        // bucket capacities: a bucket closes once fill >= cap
  uint32_t nbmax1, nbmax2;    // pool sizes in buckets (proven bounds)
  unsigned long long bsz1, bsz2;  // bucket stride in tuples = cap + tile (slack for the closing run)
  uint32_t csl;               // join slice capacity: C_R (R) or C_S (S)
  uint32_t lg2max;            // pass 2: a partition's overflow regions grow 1, 1, 2, 4, .. 2^lg2max
                              //         consecutive buckets (hj_bucket.cuh); 0 = fixed buckets
};
enum { CNT_BC_NB1 = 2, CNT_BC_NB2 = 4 };  // + relation: overflow buckets taken from the pool
constexpr uint32_t BC_LGK_SHIFT = 27, BC_J_MASK = (1u << BC_LGK_SHIFT) - 1;
constexpr uint32_t BC_MAX_NB1 = 1542;  // per relation: <= 1.5 * 2^b1 + 1 pass-1 buckets (cap1 >= 2 x mean) + prefix end + spare
enum { RES_BC_OVERFLOW = 3 };

struct Plan {
  RelDev rel[2];  // 0 = R (build), 1 = S (probe)
  int bc;         // 1: bucket-chain partitioner (NEXT-1), rel[r].t2 = bc[r].pool2
  BcRel bc_rel[2];
  int B, b1, b2;  // radix field of this plan's histogram / passes (the exchange sender: B = b1, b2 = 0)
  int g;          // rank bits in the pass-1 digit (PLAN_SEND), else 0
  int gsh;        // PLAN_SEND: the rank digit is (key >> gsh) & (2^g - 1), gsh = the local radix bits
  const uint32_t* prow[2];  // PLAN_RECV: received piece counts [nsrc][2^b1] per relation (row s = what
                            // source s sent, by pass-1 digit); rel[r].cnt is then this rank's own
                            // histogram of what it received
  int nsrc;       // count rows / piece sources (PLAN_RECV: ranks), else 1
  int mode;       // PLAN_FULL, PLAN_SEND, PLAN_RECV
  int skip_r;     // streaming S chunks: R is already partitioned (its pass-2 units are skipped)
  int pass_l2pf;  // partition passes: TMA-prefetch unit i+2's input into L2 when it is published
  int tuple_bytes;  // AoS tuple size (8 or 16): the planner zeroes each T2's 64-byte tail
  uint32_t C2;           // pass-2 chunk (tile) size in tuples
  uint32_t CR, CS;       // join item capacities: R tuples (smem build) and S tuples per item
  uint32_t lgCRp;        // log2 of the largest power of two <= CR: swapped items probe R chunks of
                         // 2^lgCRp tuples (a shift, not a division, in the planner's prefix loop)
  uint32_t* ist;         // [2^B + 1] join item prefix (q-order)
  uint32_t* ist2;        // [2^B + 1] prefix of the SWAPPED items (null: none): co-partitions whose R
                         // side needs more than one C_R chunk while S fits one (duplicate-heavy
                         // build side) are joined building on S and probing with R chunks
  uint32_t* counters;    // [8]: 0 next join item, 1 planner blocks done, 2..5 bucket-chain counters,
                         //      6 bad received counts
  unsigned long long* results;  // [4]: 0 matches, 1 checksum, 2 output cursor, 3 bucket pool overflow
  void* out_r;           // materialized payloads of R (pay width), capacity out_cap
  void* out_s;
  unsigned long long out_cap;
  unsigned long long tiles1[2];  // pass-1 tiles per relation (host-known)
  SlotHash H;            // in-partition slot hash (lg = log2 of hash-table slots per join item)
  uint32_t one;          // 1 (a runtime multiplier: keeps index * size an IMAD, see k_join)
  int mat_chk;           // MATERIALIZE also accumulates the checksum (HJ_OPT_MAT_CHECKSUM, default 1)
  __host__ __device__ int pb() const { return g + b1; }
  __host__ __device__ int qbits() const { return g + B; }
  __host__ __device__ uint32_t npieces() const { return (uint32_t)nsrc << (g + b1); }
};

// pass-1 digit D, pass-2 digit d2 and the q-order histogram bin of a key
template <bool GD, typename K>
__device__ __forceinline__ uint32_t dig1(K key, const Plan& P) {
  uint32_t d = (uint32_t)key & ((1u << P.b1) - 1);
  if (GD) d |= ((uint32_t)(key >> P.gsh) & ((1u << P.g) - 1)) << P.b1;
  return d;
}
template <typename K>
__device__ __forceinline__ uint32_t dig2(K key, const Plan& P) {
  return (uint32_t)(key >> P.b1) & ((1u << P.b2) - 1);
}
template <bool GD, typename K>
__device__ __forceinline__ uint32_t qbin(K key, const Plan& P) {
  return (dig1<GD>(key, P) << P.b2) | dig2(key, P);
}

// counters[CNT_BAD_COUNTS]: the exchange receiver's planner found count rows that do not sum
// to the tuples received (pass 2 and the join then do nothing; hj_join_received fails)
enum { CNT_NEXT_ITEM = 0, CNT_PLAN_DONE = 1, CNT_BAD_COUNTS = 6, CNT_NEXT_ITEM2 = 7 };
enum { RES_MATCHES = 0, RES_CHECKSUM = 1, RES_CURSOR = 2 };

}  // namespace hj
