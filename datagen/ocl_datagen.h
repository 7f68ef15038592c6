/*
 * ocl_datagen.h — seeded, counter-based synthetic input generators.
 *
 * This header is the ONLY code shared between the CPU oracle side (tests, bench
 * cpu_baseline) and the CUDA product side: both fill their input columns from
 * the same pure functions f(seed, field, row).  It contains NO arithmetic of the
 * method under test (no predicate, no grouping, no aggregation) — only random
 * number draws and the lineitem-shaped value recipe of SURVEY.md §8(d)
 * (distributions follow the TPC-H specification the paper cites as [36],
 * PAPER.md L1424-1426; Q1 is the paper's App. A workload).
 *
 * Every value is a pure function of (seed, global row r) so that
 *   - a GPU rank can generate its own row shard in place,
 *   - the host can regenerate exactly the same rows for the oracle,
 *   - host and device generation can be cross-checked by checksum.
 *
 * Written so it compiles as plain C99 (gcc) and as CUDA (__host__ __device__).
 */
#ifndef OCL_DATAGEN_H
#define OCL_DATAGEN_H

#include <stdint.h>

#ifdef __CUDACC__
#define OCLG_HD __host__ __device__ __forceinline__
#else
#define OCLG_HD static inline
#endif

/* Base seed: VLDB 2013 opening day; config i uses seed + i. */
#define OCLG_BASE_SEED 20130826ULL

/* Field streams (any distinct constants). */
enum {
  OCLG_F_PERM = 1, OCLG_F_ODATE = 2, OCLG_F_SHIP = 3, OCLG_F_RECEIPT = 4,
  OCLG_F_RF = 5, OCLG_F_QTY = 6, OCLG_F_PART = 7, OCLG_F_DISC = 8, OCLG_F_TAX = 9,
  OCLG_F_SW_P = 20, OCLG_F_SW_KEY = 21, OCLG_F_SW_V = 22, OCLG_F_SW_KEYHASH = 23,
  OCLG_F_FEISTEL = 30
};

#define OCLG_GOLDEN 0x9E3779B97F4A7C15ULL

/* splitmix64 output function (Steele, Lea, Flood 2014). */
OCLG_HD uint64_t oclg_mix(uint64_t z) {
  z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ULL;
  z = (z ^ (z >> 27)) * 0x94D049BB133111EBULL;
  return z ^ (z >> 31);
}

/* The ctr-th splitmix64 output of the stream (seed, field). */
OCLG_HD uint64_t oclg_u64(uint64_t seed, uint32_t field, uint64_t ctr) {
  uint64_t state = oclg_mix(seed + (uint64_t)field * OCLG_GOLDEN);
  return oclg_mix(state + (ctr + 1) * OCLG_GOLDEN);
}

/* Uniform integer in [0, range) for 1 <= range <= 2^32 (multiply-high, exact). */
OCLG_HD uint64_t oclg_below(uint64_t h, uint64_t range) {
  return ((h >> 32) * range) >> 32;
}

/* Uniform double in [0, 1) with 53 random bits (exact on host and device). */
OCLG_HD double oclg_unit(uint64_t h) {
  return (double)(h >> 11) * (1.0 / 9007199254740992.0);
}

/* ---------------------------------------------------------------- lineitem */

/* Dates are int32 days since 1970-01-01. */
#define OCLG_DATE_1992_01_01 8035
#define OCLG_ODATE_SPAN 2406          /* orderdate ~ U[8035, 10440] */
#define OCLG_DATE_1995_06_17 9298     /* linestatus / returnflag cutoff */
#define OCLG_Q1_SHIP_CUTOFF 10471     /* date '1998-12-01' - 90 days */

typedef struct {
  int64_t orderkey;
  int32_t shipdate;
  uint8_t returnflag;
  uint8_t linestatus;
  int64_t quantity;       /* decimal, scale 2 (100 == 1.00) */
  int64_t extendedprice;  /* decimal, scale 2 */
  int64_t discount;       /* decimal, scale 2: 0..10 == 0.00..0.10 */
  int64_t tax;            /* decimal, scale 2: 0..8 */
} oclg_lineitem_row;

/* Orders: blocks of 28 consecutive rows hold 7 orders whose line counts are a
 * seeded permutation of {1..7}.  Returns the global order index of row r. */
OCLG_HD uint64_t oclg_order_of_row(uint64_t seed, uint64_t r) {
  uint64_t b = r / 28, off = r % 28;
  int len[7] = {1, 2, 3, 4, 5, 6, 7};
  for (int i = 6; i > 0; --i) {           /* Fisher-Yates, 6 draws */
    uint64_t j = oclg_below(oclg_u64(seed, OCLG_F_PERM, b * 8 + (uint64_t)i), (uint64_t)(i + 1));
    int t = len[i]; len[i] = len[j]; len[j] = t;
  }
  uint64_t acc = 0;
  int k = 0;
  for (; k < 6; ++k) {
    acc += (uint64_t)len[k];
    if (off < acc) break;
  }
  return b * 7 + (uint64_t)k;
}

OCLG_HD oclg_lineitem_row oclg_lineitem(uint64_t seed, uint64_t r, uint64_t nparts) {
  oclg_lineitem_row x;
  uint64_t o = oclg_order_of_row(seed, r);
  x.orderkey = (int64_t)((o / 8) * 32 + o % 8 + 1);
  int32_t odate = OCLG_DATE_1992_01_01 + (int32_t)oclg_below(oclg_u64(seed, OCLG_F_ODATE, o), OCLG_ODATE_SPAN);
  int32_t ship = odate + 1 + (int32_t)oclg_below(oclg_u64(seed, OCLG_F_SHIP, r), 121);
  int32_t receipt = ship + 1 + (int32_t)oclg_below(oclg_u64(seed, OCLG_F_RECEIPT, r), 30);
  x.shipdate = ship;
  x.linestatus = (uint8_t)(ship > OCLG_DATE_1995_06_17 ? 'O' : 'F');
  if (receipt > OCLG_DATE_1995_06_17) x.returnflag = (uint8_t)'N';
  else x.returnflag = (uint8_t)(oclg_below(oclg_u64(seed, OCLG_F_RF, r), 2) ? 'R' : 'A');
  int64_t units = 1 + (int64_t)oclg_below(oclg_u64(seed, OCLG_F_QTY, r), 50);
  int64_t pk = 1 + (int64_t)oclg_below(oclg_u64(seed, OCLG_F_PART, r), nparts);
  int64_t retail = 90000 + ((pk / 10) % 20001) + 100 * (pk % 1000);
  x.quantity = 100 * units;
  x.extendedprice = units * retail;
  x.discount = (int64_t)oclg_below(oclg_u64(seed, OCLG_F_DISC, r), 11);
  x.tax = (int64_t)oclg_below(oclg_u64(seed, OCLG_F_TAX, r), 9);
  return x;
}

/* nparts for scale factor sf: SF * 200000 parts (at least 1). */
OCLG_HD uint64_t oclg_nparts_for_rows(uint64_t n) {
  /* n = SF * 6,000,000  =>  SF * 200,000 = n / 30 */
  uint64_t p = n / 30;
  return p ? p : 1;
}

/* Seeded Feistel permutation of [0, n) (cycle walking over a power-of-4
 * domain); used for the "shuffled" row order of config C3. */
OCLG_HD uint64_t oclg_feistel(uint64_t seed, uint64_t n, uint64_t x) {
  int half = 1;
  while ((1ULL << (2 * half)) < n) ++half;
  uint64_t mask = (1ULL << half) - 1;
  do {
    uint64_t L = x >> half, R = x & mask;
    for (int round = 0; round < 4; ++round) {
      uint64_t F = oclg_u64(seed, OCLG_F_FEISTEL, (R << 3) | (uint64_t)round) & mask;
      uint64_t t = L ^ F; L = R; R = t;
    }
    x = (L << half) | R;
  } while (x >= n);
  return x;
}

/* ------------------------------------------------------ cardinality sweep C5 */

/* p ~ U[0, 10^6) (int32), v ~ U[0, 10^6) (int64), key = mix(rank ^ seed')
 * with rank ~ Zipf(s) over G ranks via an inverse-CDF table (s = 0: uniform,
 * cdf == NULL). cdf[i] = P(rank <= i), cdf[G-1] == 1.0 exactly. */
OCLG_HD int32_t oclg_sweep_p(uint64_t seed, uint64_t r) {
  return (int32_t)oclg_below(oclg_u64(seed, OCLG_F_SW_P, r), 1000000);
}
OCLG_HD int64_t oclg_sweep_v(uint64_t seed, uint64_t r) {
  return (int64_t)oclg_below(oclg_u64(seed, OCLG_F_SW_V, r), 1000000);
}
OCLG_HD uint64_t oclg_sweep_rank(uint64_t seed, uint64_t r, uint64_t G, const double* cdf) {
  uint64_t h = oclg_u64(seed, OCLG_F_SW_KEY, r);
  if (!cdf) return oclg_below(h, G);
  double u = oclg_unit(h);
  uint64_t lo = 0, hi = G - 1;          /* smallest i with u < cdf[i] */
  while (lo < hi) {
    uint64_t mid = (lo + hi) >> 1;
    if (u < cdf[mid]) hi = mid; else lo = mid + 1;
  }
  return lo;
}
OCLG_HD int64_t oclg_sweep_key(uint64_t seed, uint64_t rank) {
  return (int64_t)oclg_mix(rank ^ oclg_u64(seed, OCLG_F_SW_KEYHASH, 0));
}

#endif /* OCL_DATAGEN_H */
