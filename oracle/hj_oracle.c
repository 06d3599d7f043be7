/*
 * hj_oracle.c -- TEST INFRASTRUCTURE ONLY. The plain, slow, obviously-correct CPU
 * oracle for the radix-partitioned hash join of Sioulas et al. (ICDE 2019).
 *
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline / --impl reference
 * legs may load this library. The product path (paper_conf_icde_sioulasckaa19_b200/)
 * never links, imports or calls it, and it shares no code with csrc/: it uses a
 * different hash (Fibonacci multiplicative hashing on the whole key, not the GPU's
 * low-bit radix digits) and no blocking, fusion or reordering.
 *
 * Single-threaded, no OpenMP. Citations are PAPER.md line ranges ("P:a-b").
 *
 * Result definition (reading S1-S4 of §8(c.4)):
 *   J        = multiset {(r_pay, s_pay) : r_key == s_key}   (bag semantics)
 *   matches  = |J| (uint64)
 *   checksum = sum over J of sig(r_pay, s_pay) mod 2^64
 *   sig(p,q) = fmix64(p ^ (q * 0x9E3779B97F4A7C15)), payloads zero-extended to 64 bits,
 *              fmix64 = the splitmix64 finalizer (pinned by tests/golden/splitmix64.txt).
 *
 * Pins (tests/test_oracle.py): brute-force nested loop on small inputs, numpy sort-merge
 * count, closed forms of the generator (FK / 1:1 joins have exactly |S| matches and
 * checksum sum_j sig(rho(j), j)), the hand-worked example in tests/golden/, and the
 * splitmix64 published outputs.
 */
#include <stdint.h>
#include <stdlib.h>
#include <string.h>

#define ORACLE_OK 0
#define ORACLE_ERR_INVALID (-1)
#define ORACLE_ERR_OOM (-3)

static uint64_t fmix64(uint64_t z) {
  z ^= z >> 30;
  z *= 0xBF58476D1CE4E5B9ULL;
  z ^= z >> 27;
  z *= 0x94D049BB133111EBULL;
  z ^= z >> 31;
  return z;
}

/* Pair signature of one join result (reading S1). */
uint64_t oracle_sig(uint64_t r_pay, uint64_t s_pay) {
  return fmix64(r_pay ^ (s_pay * 0x9E3779B97F4A7C15ULL));
}

uint64_t oracle_fmix64(uint64_t z) { return fmix64(z); }

static uint64_t load_col(const void* col, int bytes, uint64_t i) {
  if (bytes == 4) return (uint64_t)((const uint32_t*)col)[i];
  return ((const uint64_t*)col)[i];
}

static void store_col(void* col, int bytes, uint64_t i, uint64_t v) {
  if (bytes == 4) ((uint32_t*)col)[i] = (uint32_t)v;
  else ((uint64_t*)col)[i] = v;
}

/* A key belongs to slice t of 2^slice_bits iff the top slice_bits of fmix64(key) equal t.
 * The join decomposes exactly over any partition of the key domain. */
static int in_slice(uint64_t key, int slice_bits, uint64_t slice_id) {
  if (slice_bits <= 0) return 1;
  return (fmix64(key) >> (64 - slice_bits)) == slice_id;
}

/*
 * The canonical hash join (§II-B): build a hash table on R, then probe it
 * with every tuple of S. Chained table: head[nb] and next[nR] as row indices.
 *
 *   1. nb = next power of two >= max(nR, 1); head[] = NIL.
 *   2. for i in 0..nR-1: h = (k_i * 0x9E3779B97F4A7C15) >> (64 - log2 nb); next[i] = head[h]; head[h] = i
 *   3. for j in 0..nS-1: walk i = head[h(k'_j)] via next; on k_i == k'_j count, add sig, append pair
 *
 * out_r / out_s may be NULL (no materialization); otherwise at most `cap` pairs are
 * written (in probe order) and `matches` still counts all of them.
 * Returns ORACLE_OK, ORACLE_ERR_INVALID or ORACLE_ERR_OOM.
 */
int oracle_hash_join(int key_bytes, int pay_bytes,
                     const void* R_keys, const void* R_pay, uint64_t nR,
                     const void* S_keys, const void* S_pay, uint64_t nS,
                     int slice_bits, uint64_t slice_id,
                     void* out_r, void* out_s, uint64_t cap,
                     uint64_t* matches_out, uint64_t* checksum_out) {
  if ((key_bytes != 4 && key_bytes != 8) || (pay_bytes != 4 && pay_bytes != 8)) return ORACLE_ERR_INVALID;
  if (!matches_out || !checksum_out) return ORACLE_ERR_INVALID;
  *matches_out = 0;
  *checksum_out = 0;
  if (nR == 0 || nS == 0) return ORACLE_OK;
  if (!R_keys || !R_pay || !S_keys || !S_pay) return ORACLE_ERR_INVALID;

  int lg = 0;
  while ((1ULL << lg) < nR) ++lg;
  if (lg == 0) lg = 1; /* one-row R: a 2-slot table keeps the shift below 64 */
  const uint64_t nb = 1ULL << lg;
  const uint64_t NIL = UINT64_MAX;
  uint64_t* head = (uint64_t*)malloc(nb * sizeof(uint64_t));
  uint64_t* next = (uint64_t*)malloc(nR * sizeof(uint64_t));
  if (!head || !next) {
    free(head);
    free(next);
    return ORACLE_ERR_OOM;
  }
  for (uint64_t h = 0; h < nb; ++h) head[h] = NIL;

  /* build phase */
  for (uint64_t i = 0; i < nR; ++i) {
    uint64_t k = load_col(R_keys, key_bytes, i);
    if (!in_slice(k, slice_bits, slice_id)) continue;
    uint64_t h = (k * 0x9E3779B97F4A7C15ULL) >> (64 - lg);
    next[i] = head[h];
    head[h] = i;
  }

  /* probe phase */
  uint64_t matches = 0, checksum = 0;
  for (uint64_t j = 0; j < nS; ++j) {
    uint64_t k = load_col(S_keys, key_bytes, j);
    if (!in_slice(k, slice_bits, slice_id)) continue;
    uint64_t q = load_col(S_pay, pay_bytes, j);
    uint64_t h = (k * 0x9E3779B97F4A7C15ULL) >> (64 - lg);
    for (uint64_t i = head[h]; i != NIL; i = next[i]) {
      if (load_col(R_keys, key_bytes, i) != k) continue;
      uint64_t p = load_col(R_pay, pay_bytes, i);
      if (out_r && out_s && matches < cap) {
        store_col(out_r, pay_bytes, matches, p);
        store_col(out_s, pay_bytes, matches, q);
      }
      ++matches;
      checksum += oracle_sig(p, q);
    }
  }
  free(head);
  free(next);
  *matches_out = matches;
  *checksum_out = checksum;
  return ORACLE_OK;
}

/*
 * Radix partitioning, plain definition (Fig. 1; reading S5): tuple (k, v) goes
 * to partition p = (k >> shift) & (2^bits - 1). Output = a stable counting sort by p:
 *   counts[p] = #tuples with digit p; offsets = exclusive prefix sum of counts (offsets[2^bits] = n);
 *   tuples are copied in input order to out[offsets[p] + (#earlier tuples with digit p)].
 * Any correct partitioner yields the same MULTISET of tuples in every partition; this one
 * additionally fixes the order inside a partition (stable), which np.argsort(kind='stable')
 * pins in tests.
 */
int oracle_radix_partition(int key_bytes, int pay_bytes,
                           const void* keys, const void* pays, uint64_t n,
                           int shift, int bits,
                           void* out_keys, void* out_pays, uint64_t* offsets /* 2^bits + 1 */) {
  if ((key_bytes != 4 && key_bytes != 8) || (pay_bytes != 4 && pay_bytes != 8)) return ORACLE_ERR_INVALID;
  if (bits < 0 || bits > 24 || shift < 0 || shift >= 8 * key_bytes || !offsets) return ORACLE_ERR_INVALID;
  const uint64_t np_ = 1ULL << bits;
  const uint64_t mask = np_ - 1;
  uint64_t* cursor = (uint64_t*)calloc(np_, sizeof(uint64_t));
  if (!cursor) return ORACLE_ERR_OOM;
  memset(offsets, 0, (np_ + 1) * sizeof(uint64_t));
  for (uint64_t i = 0; i < n; ++i) offsets[((load_col(keys, key_bytes, i) >> shift) & mask) + 1] += 1;
  for (uint64_t p = 0; p < np_; ++p) offsets[p + 1] += offsets[p];
  for (uint64_t p = 0; p < np_; ++p) cursor[p] = offsets[p];
  for (uint64_t i = 0; i < n; ++i) {
    uint64_t k = load_col(keys, key_bytes, i);
    uint64_t p = (k >> shift) & mask;
    uint64_t dst = cursor[p]++;
    store_col(out_keys, key_bytes, dst, k);
    store_col(out_pays, pay_bytes, dst, load_col(pays, pay_bytes, i));
  }
  free(cursor);
  return ORACLE_OK;
}
