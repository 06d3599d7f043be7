// hj_plan.cuh -- device-side plan shared by all kernels of one hj_join call.
#pragma once
#include <cstdint>

#include "hj_common.cuh"

namespace hj {

// Per-relation device state. Co-partition q-order: q = d1 << b2 | d2 where the key's radix
// field p = key & (2^B - 1) splits into d1 = p & (2^b1 - 1) (pass 1) and d2 = p >> b1 (pass 2).
// Partition d1 of pass 1 is then the contiguous q range [d1 << b2, (d1 + 1) << b2).
struct RelDev {
  const void* keys;  // SoA input (caller-owned)
  const void* pays;
  unsigned long long n;
  void* t1;                   // pass-1 output, AoS, n tuples
  void* t2;                   // pass-2 output, AoS, n tuples, co-partitions contiguous in q-order
  uint32_t* cnt;              // [2^B] histogram, q-order (k_hist translates p -> q)
  unsigned long long* off;    // [2^B + 1] co-partition start, q-order (exclusive scan)
  unsigned long long* cur1;   // [2^b1] pass-1 reservation cursors
  unsigned long long* cur2;   // [2^B]  pass-2 reservation cursors (q-order)
  uint32_t* cst;              // [2^b1 + 1] pass-2 chunk prefix (chunks of C2 tuples per d1)
};

struct Plan {
  RelDev rel[2];  // 0 = R (build), 1 = S (probe)
  int B, b1, b2;
  uint32_t C2;           // pass-2 chunk (tile) size in tuples
  uint32_t CR, CS;       // join item capacities: R tuples (smem build) and S tuples per item
  uint32_t* ist;         // [2^B + 1] join item prefix (q-order)
  uint32_t* counters;    // [8]: 0 next join item, 1 planner blocks done, 2.. reserved
  unsigned long long* results;  // [4]: 0 matches, 1 checksum, 2 output cursor, 3 unused
  void* out_r;           // materialized payloads of R (pay width), capacity out_cap
  void* out_s;
  unsigned long long out_cap;
  unsigned long long tiles1[2];  // pass-1 tiles per relation (host-known)
  SlotHash H;            // in-partition slot hash (lg = log2 of hash-table slots per join item)
};

enum { CNT_NEXT_ITEM = 0, CNT_PLAN_DONE = 1 };
enum { RES_MATCHES = 0, RES_CHECKSUM = 1, RES_CURSOR = 2 };

}  // namespace hj
