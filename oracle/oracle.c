/*
 * oracle.c -- TEST INFRASTRUCTURE ONLY.
 *
 * Plain, slow, obviously-correct CPU oracle for the equi-join micro-benchmark
 * of PAPER.md §6.2 (P789-794): "two equally-sized tables, each with two 4-byte
 * columns: a key and a payload ... an equi-join over the key columns that is
 * followed by a sum/count aggregation over each payload column".
 *
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline /
 * --impl reference legs may load this library.  It shares no code, header,
 * constant table or helper with the CUDA product path
 * (paper_conf_cidr_chrysogelossa19_b200/csrc); neither includes the other.
 *
 * What it computes is the plain definition of the result, not the paper's
 * algorithm (the radix join reaches exactly this result faster):
 *   J = { (p_i, q_j) : k_i == k'_j }        (inner equi-join, bag semantics,
 *                                            key equality = bit equality)
 *   match_count   = |J|
 *   sum_r         = sum over J of (u64)(i64) p      (mod 2^64)
 *   sum_s         = sum over J of (u64)(i64) q      (mod 2^64)
 *   pair_checksum = sum over J of mix(p, q)         (mod 2^64)
 *   mix(p, q)     = fmix64((u64)p * 0x9E3779B97F4A7C15 + (u64)q)
 *   fmix64        = the splitmix64 finaliser
 * Readings of the paper's silences (bag semantics, sign extension, wrapping
 * u64 sums, pair_checksum itself) are DESIGN.md readings R5/R6/R8/R10.
 *
 * Algorithm: copy both sides into (key, payload) arrays,
 * qsort each by key, merge; for each equal-key run of a R rows and b S rows
 * add a*b to the count, b*sum(run_R p) and a*sum(run_S q) to the sums, and
 * visit all a*b pairs for the checksum / materialisation.  Materialised pairs
 * are finally qsorted lexicographically as signed (p, q).
 */
#include <stdint.h>
#include <stdlib.h>
#include <string.h>

typedef struct { int64_t k; int64_t p; } oracle_tuple;

static uint64_t oracle_fmix64(uint64_t x) {
  x ^= x >> 30; x *= 0xbf58476d1ce4e5b9ULL;
  x ^= x >> 27; x *= 0x94d049bb133111ebULL;
  x ^= x >> 31;
  return x;
}

uint64_t oracle_mix(int64_t p, int64_t q) {
  return oracle_fmix64((uint64_t)p * 0x9E3779B97F4A7C15ULL + (uint64_t)q);
}

uint64_t oracle_fmix64_export(uint64_t x) { return oracle_fmix64(x); }

static int64_t load_signed(const void* col, int bytes, uint64_t i) {
  if (bytes == 4) return (int64_t)((const int32_t*)col)[i];
  return ((const int64_t*)col)[i];
}

static int cmp_key(const void* a, const void* b) {
  int64_t x = ((const oracle_tuple*)a)->k, y = ((const oracle_tuple*)b)->k;
  return (x > y) - (x < y);
}

static int cmp_pair(const void* a, const void* b) {
  const oracle_tuple* x = (const oracle_tuple*)a;
  const oracle_tuple* y = (const oracle_tuple*)b;
  if (x->k != y->k) return (x->k > y->k) - (x->k < y->k);
  return (x->p > y->p) - (x->p < y->p);
}

/*
 * oracle_join: returns 0 on success, -1 on bad arguments / allocation failure.
 *   key_bytes, rp_bytes, sp_bytes in {4, 8}; columns are host arrays.
 *   out[0..3] = match_count, sum_r, sum_s, pair_checksum.
 *   If pairs_r/pairs_s are non-NULL, up to pairs_cap pairs are written sorted
 *   lexicographically by (p, q) as signed int64; *n_pairs = |J| always.
 *   (Sorting is over the first min(|J|, pairs_cap) pairs emitted only when
 *   |J| <= pairs_cap; otherwise the written prefix is unsorted and the caller
 *   must treat it as invalid.)
 */
int oracle_join(int key_bytes,
                const void* rk, const void* rp, int rp_bytes, uint64_t nr,
                const void* sk, const void* sp, int sp_bytes, uint64_t ns,
                uint64_t out[4],
                int64_t* pairs_r, int64_t* pairs_s, uint64_t pairs_cap,
                uint64_t* n_pairs) {
  if ((key_bytes != 4 && key_bytes != 8) || (rp_bytes != 4 && rp_bytes != 8) ||
      (sp_bytes != 4 && sp_bytes != 8) || !out)
    return -1;
  out[0] = out[1] = out[2] = out[3] = 0;
  if (n_pairs) *n_pairs = 0;
  oracle_tuple* R = (oracle_tuple*)malloc((nr ? nr : 1) * sizeof(oracle_tuple));
  oracle_tuple* S = (oracle_tuple*)malloc((ns ? ns : 1) * sizeof(oracle_tuple));
  if (!R || !S) { free(R); free(S); return -1; }
  /* step 1: copy; step 2: sort both sides by key */
  for (uint64_t i = 0; i < nr; i++) { R[i].k = load_signed(rk, key_bytes, i); R[i].p = load_signed(rp, rp_bytes, i); }
  for (uint64_t j = 0; j < ns; j++) { S[j].k = load_signed(sk, key_bytes, j); S[j].p = load_signed(sp, sp_bytes, j); }
  qsort(R, nr, sizeof(oracle_tuple), cmp_key);
  qsort(S, ns, sizeof(oracle_tuple), cmp_key);
  /* step 3: merge */
  uint64_t cnt = 0, sr = 0, ss = 0, sx = 0, w = 0;
  uint64_t i = 0, j = 0;
  while (i < nr && j < ns) {
    if (R[i].k < S[j].k) { i++; continue; }
    if (R[i].k > S[j].k) { j++; continue; }
    int64_t key = R[i].k;
    uint64_t i1 = i, j1 = j, sum_rp = 0, sum_sp = 0;
    while (i1 < nr && R[i1].k == key) { sum_rp += (uint64_t)R[i1].p; i1++; }
    while (j1 < ns && S[j1].k == key) { sum_sp += (uint64_t)S[j1].p; j1++; }
    uint64_t a = i1 - i, b = j1 - j;
    cnt += a * b;
    sr += b * sum_rp;
    ss += a * sum_sp;
    for (uint64_t x = i; x < i1; x++)
      for (uint64_t y = j; y < j1; y++) {
        sx += oracle_mix(R[x].p, S[y].p);
        if (pairs_r && pairs_s && w < pairs_cap) { pairs_r[w] = R[x].p; pairs_s[w] = S[y].p; }
        w++;
      }
    i = i1; j = j1;
  }
  out[0] = cnt; out[1] = sr; out[2] = ss; out[3] = sx;
  if (n_pairs) *n_pairs = cnt;
  free(R); free(S);
  /* step 4: sort the materialised pairs */
  if (pairs_r && pairs_s && cnt <= pairs_cap && cnt > 0) {
    oracle_tuple* P = (oracle_tuple*)malloc(cnt * sizeof(oracle_tuple));
    if (!P) return -1;
    for (uint64_t x = 0; x < cnt; x++) { P[x].k = pairs_r[x]; P[x].p = pairs_s[x]; }
    qsort(P, cnt, sizeof(oracle_tuple), cmp_pair);
    for (uint64_t x = 0; x < cnt; x++) { pairs_r[x] = P[x].k; pairs_s[x] = P[x].p; }
    free(P);
  }
  return 0;
}
