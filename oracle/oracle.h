/*
 * oracle.h — TEST INFRASTRUCTURE ONLY.
 *
 * A plain, slow, obviously-correct, single-threaded CPU implementation of the
 * Ocelot select -> hash GROUP BY -> aggregate path (Heimel et al., PVLDB 6(9)
 * 2013, §4.1), written from the paper's operator
 * definitions and SURVEY.md §8(c).  It shares NO code with the CUDA product
 * path (paper_journals_pvldb_heimelspmm13_b200/csrc): its own types, its own
 * constants, its own hashing (std::unordered_map).  Only tests/,
 * __graft_entry__.smoke() and bench.py's cpu_baseline / --impl reference leg
 * may load it.
 *
 * Pins (tests/test_oracle_*.py): brute-force predicate and nested-loop grouping
 * in pure Python, hash-vs-sort grouping equality, closed forms for keys r mod G
 * and values r, exact-integer pin of fp64 sums, the hand-computed Q1 worked
 * example (tests/golden/q1_worked_example.txt), invariants.
 * Parity unpinned: none of the functions below (GPU gid *labels* and fp64
 * bit patterns are unpinned by design; only the partition and the tolerance
 * are compared).
 */
#ifndef OCELOT_ORACLE_H
#define OCELOT_ORACLE_H

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

/* dtype codes (numerically equal to the product ABI's, but defined here). */
enum { ORC_U8 = 1, ORC_I32 = 2, ORC_I64 = 3, ORC_F64 = 4 };

typedef struct {
  const void* data;
  int32_t dtype;
  int32_t pad_;
  int64_t n;
} orc_column;

/* MonetDB-style range predicate: per-side inclusive flags,
 * unbounded sides, anti.  Integer bounds in lo_i/hi_i, fp64 bounds in lo_f/hi_f. */
typedef struct {
  int32_t dtype;
  uint8_t has_lo, has_hi, lo_incl, hi_incl;
  uint8_t anti, pad_[7];
  int64_t lo_i, hi_i;
  double lo_f, hi_f;
} orc_range;

enum { ORC_AGG_COUNT = 0, ORC_AGG_SUM = 1, ORC_AGG_MIN = 2, ORC_AGG_MAX = 3, ORC_AGG_AVG = 4 };
enum { ORC_EXPR_COL = 0, ORC_EXPR_MUL_1MINUS = 1, ORC_EXPR_MUL_1MINUS_1PLUS = 2 };

typedef struct {
  int32_t op, expr;
  int32_t a, b, c;         /* indices into vals[]; a = -1 for COUNT(*) */
  int32_t decimal_scale;   /* S = 10^scale is "1" in the expressions */
  void* out;               /* [G]; layout per op, see oracle_aggregate */
} orc_agg;

/* a1: bitmap[r>>5] bit (r&31) = pred(col[r]); ceil(n/32)
 * words, tail bits zero.  Returns 0 on success, -1 on bad dtype. */
int oracle_select(const orc_column* col, const orc_range* pred, uint32_t* bitmap);
/* A2 (L435-438): out = a OP b over ceil(n/32) words; op 0 AND, 1 OR, 2 ANDNOT (a & ~b). */
void oracle_bitmap_combine(int op, const uint32_t* a, const uint32_t* b, uint32_t* out, int64_t n);
/* a2 (L449-455): ascending row ids of set bits; returns m. */
int64_t oracle_compact(const uint32_t* bitmap, int64_t n, uint32_t* oids);
/* a3 (L443-449): out[j] = col[oids[j]] (element size from dtype). */
void oracle_gather(const orc_column* col, const uint32_t* oids, int64_t m, void* out);
/* a4-a6 (L551-561): packed key of row r (nkeys 1 or 2, raw bits zero-extended,
 * key = a << width(b) | b).  Dense gids by FIRST OCCURRENCE in oid order
 * (MonetDB group.group).  oids == NULL means rows 0..m-1.  Returns G, or -1 on
 * invalid key spec.  keys_out[g] = packed key of group g. */
int64_t oracle_group_hash(const orc_column* keys, int nkeys, const uint32_t* oids, int64_t m,
                          int32_t* gids, int64_t* keys_out);
/* Independent second implementation: stable sort of (key, j) -> runs -> gid by
 * min j of each run.  Must equal oracle_group_hash exactly. */
int64_t oracle_group_sort(const orc_column* keys, int nkeys, const uint32_t* oids, int64_t m,
                          int32_t* gids, int64_t* keys_out);
/* a4, sorted input (L554-556 §4.1.6): successor compare marks group ends, an
 * exclusive prefix sum of the marks is the dense gid (group g = g-th distinct key
 * in row order).  Returns G, -1 on invalid key spec, -2 if the packed key
 * (unsigned) decreases anywhere (input not sorted). */
int64_t oracle_group_sorted(const orc_column* keys, int nkeys, const uint32_t* oids, int64_t m,
                            int32_t* gids, int64_t* keys_out);
/* Equi hash join (L534-550 §4.1.5): all pairs (probe row, build row) with equal keys
 * (one integer key column per side, same dtype), in probe order, partners ascending.
 * probe rows j < m at oids[j] (NULL: row j).  Returns the pair count (pairs written while
 * < out_capacity), -1 on an invalid spec. */
int64_t oracle_hash_join(const orc_column* build, const orc_column* probe, const uint32_t* oids, int64_t m,
                         uint32_t* out_probe, uint32_t* out_build, int64_t out_capacity);
/* a7-a8 (L562-568): per group g in [0,G):
 *   COUNT -> int64;  SUM over int64 (expr values in int128, wrapping mod 2^128)
 *   -> 16 bytes {uint64 lo, int64 hi};  SUM over f64 -> double (Neumaier
 *   compensated);  MIN/MAX -> input dtype (int64 / double);  AVG -> double =
 *   (double)SUM / (double)COUNT.  Values are read at vals[k].data[oids[j]]
 *   (oids == NULL: row j).  Returns 0, or -1 on invalid spec. */
int oracle_aggregate(const int32_t* gids, const uint32_t* oids, int64_t m, int64_t G,
                     const orc_column* vals, int nvals, const orc_agg* aggs, int naggs);
/* a9: the composition select(conjunction of npreds) -> compact -> group ->
 * aggregate.  npreds == 0 selects all rows; nkeys == 0 is one group (key 0)
 * when at least one row qualifies.  order_by_key sorts output rows by the
 * packed key (unsigned).  Returns G (>= 0), or -1 on invalid spec, or -2 if
 * G > out_capacity (nothing written). */
int64_t oracle_sga(const orc_column* pred_cols, const orc_range* preds, int npreds,
                   const orc_column* key_cols, int nkeys, const orc_column* vals, int nvals,
                   const orc_agg* aggs, int naggs, int order_by_key, int64_t* keys_out,
                   int64_t out_capacity);

#ifdef __cplusplus
}
#endif
#endif
