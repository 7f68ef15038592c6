// oracle.cpp — TEST INFRASTRUCTURE ONLY (see oracle.h for scope and pins).
//
// Plain single-threaded C++17.  Every function is the textbook definition of
// one step of Ocelot's select -> group -> aggregate path, in the paper's order
// (§4.1.1 selection L429-438, §4.1.2 projection/bitmap->TIDs L443-455,
// §4.1.6 group-by L551-561, §4.1.7 aggregation L562-568) with the readings of
// SURVEY.md §8(c) (s1-s20) where the paper is silent.  No blocking, no fusion,
// no tuning.  Compiled with -O2 -ffp-contract=off (no FMA contraction, so each
// fp64 row expression is evaluated left to right, s14).
#include "oracle.h"

#include <algorithm>
#include <cmath>
#include <cstring>
#include <unordered_map>
#include <utility>
#include <vector>

namespace {

typedef unsigned __int128 u128;
typedef __int128 i128;

int elem_size(int dtype) {
  switch (dtype) {
    case ORC_U8: return 1;
    case ORC_I32: return 4;
    case ORC_I64: return 8;
    case ORC_F64: return 8;
    default: return 0;
  }
}

// Raw bits of element r zero-extended to 64 (key packing, s5).
uint64_t raw_bits(const orc_column& c, int64_t r) {
  switch (c.dtype) {
    case ORC_U8: return ((const uint8_t*)c.data)[r];
    case ORC_I32: return (uint32_t)((const int32_t*)c.data)[r];
    case ORC_I64: return (uint64_t)((const int64_t*)c.data)[r];
    case ORC_F64: { uint64_t u; std::memcpy(&u, (const double*)c.data + r, 8); return u; }
  }
  return 0;
}

int64_t int_value(const orc_column& c, int64_t r) {
  switch (c.dtype) {
    case ORC_U8: return ((const uint8_t*)c.data)[r];
    case ORC_I32: return ((const int32_t*)c.data)[r];
    case ORC_I64: return ((const int64_t*)c.data)[r];
  }
  return 0;
}

double f64_value(const orc_column& c, int64_t r) { return ((const double*)c.data)[r]; }

// s2: pred(x) = (!has_lo || (lo_incl ? x >= lo : x > lo)) && (!has_hi || (hi_incl ? x <= hi : x < hi)), XOR anti.
template <class T>
bool range_pred(T x, bool has_lo, T lo, bool lo_incl, bool has_hi, T hi, bool hi_incl, bool anti) {
  bool ok = true;
  if (has_lo) ok = ok && (lo_incl ? x >= lo : x > lo);
  if (has_hi) ok = ok && (hi_incl ? x <= hi : x < hi);
  return anti ? !ok : ok;
}

bool row_pred(const orc_column& c, const orc_range& p, int64_t r) {
  if (c.dtype == ORC_F64)
    return range_pred<double>(f64_value(c, r), p.has_lo, p.lo_f, p.lo_incl, p.has_hi, p.hi_f, p.hi_incl, p.anti);
  return range_pred<int64_t>(int_value(c, r), p.has_lo, p.lo_i, p.lo_incl, p.has_hi, p.hi_i, p.hi_incl, p.anti);
}

bool keys_valid(const orc_column* keys, int nkeys) {
  if (nkeys < 1 || nkeys > 2) return false;
  int bits = 0;
  for (int k = 0; k < nkeys; ++k) {
    if (keys[k].dtype == ORC_F64 || elem_size(keys[k].dtype) == 0) return false;
    bits += 8 * elem_size(keys[k].dtype);
  }
  return bits <= 64;
}

// s5: key = zext(a) << width(b) | zext(b).
uint64_t packed_key(const orc_column* keys, int nkeys, int64_t r) {
  if (nkeys == 1) return raw_bits(keys[0], r);
  int wb = 8 * elem_size(keys[1].dtype);
  return (raw_bits(keys[0], r) << wb) | raw_bits(keys[1], r);
}

// Neumaier-compensated summation (the fp64 SUM reference).
struct Neumaier {
  double s = 0.0, c = 0.0;
  void add(double x) {
    double t = s + x;
    if (std::fabs(s) >= std::fabs(x)) c += (s - t) + x;
    else c += (x - t) + s;
    s = t;
  }
  double value() const { return s + c; }
};

bool is_f64(const orc_column* vals, int idx) { return vals[idx].dtype == ORC_F64; }

// Validate one aggregate spec against the value columns.
bool agg_valid(const orc_agg& g, const orc_column* vals, int nvals) {
  if (g.op == ORC_AGG_COUNT) return g.a < nvals;
  if (g.op < 0 || g.op > ORC_AGG_AVG) return false;
  if (g.a < 0 || g.a >= nvals) return false;
  if (vals[g.a].dtype == ORC_U8) return false;
  int need = g.expr == ORC_EXPR_COL ? 1 : (g.expr == ORC_EXPR_MUL_1MINUS ? 2 : (g.expr == ORC_EXPR_MUL_1MINUS_1PLUS ? 3 : -1));
  if (need < 0) return false;
  if ((g.op == ORC_AGG_MIN || g.op == ORC_AGG_MAX) && g.expr != ORC_EXPR_COL) return false;
  int idx[3] = {g.a, g.b, g.c};
  for (int k = 1; k < need; ++k) {
    if (idx[k] < 0 || idx[k] >= nvals) return false;
    if (vals[idx[k]].dtype == ORC_U8) return false;
    if (is_f64(vals, idx[k]) != is_f64(vals, g.a)) return false;   // no mixed int/fp expressions
  }
  if (g.decimal_scale < 0 || g.decimal_scale > 18) return false;
  return true;
}

int64_t pow10_i(int s) { int64_t v = 1; for (int i = 0; i < s; ++i) v *= 10; return v; }

// Integer expression value in int128, wrapping mod 2^128 (the ABI's definition).
u128 int_expr(const orc_agg& g, const orc_column* vals, int64_t r) {
  u128 S = (u128)(i128)pow10_i(g.decimal_scale);
  u128 a = (u128)(i128)int_value(vals[g.a], r);
  if (g.expr == ORC_EXPR_COL) return a;
  u128 b = (u128)(i128)int_value(vals[g.b], r);
  u128 e = a * (S - b);
  if (g.expr == ORC_EXPR_MUL_1MINUS) return e;
  u128 c = (u128)(i128)int_value(vals[g.c], r);
  return e * (S + c);
}

// fp64 expression value: (a * (S - b)) * (S + c), left to right, S = 10^scale.
double f64_expr(const orc_agg& g, const orc_column* vals, int64_t r) {
  double S = (double)pow10_i(g.decimal_scale);
  double a = f64_value(vals[g.a], r);
  if (g.expr == ORC_EXPR_COL) return a;
  double b = f64_value(vals[g.b], r);
  double e = a * (S - b);
  if (g.expr == ORC_EXPR_MUL_1MINUS) return e;
  double c = f64_value(vals[g.c], r);
  return e * (S + c);
}

size_t out_elem_bytes(const orc_agg& g, const orc_column* vals) {
  if (g.op == ORC_AGG_SUM && !is_f64(vals, g.a)) return 16;
  return 8;
}

}  // namespace

extern "C" {

int oracle_select(const orc_column* col, const orc_range* pred, uint32_t* bitmap) {
  if (elem_size(col->dtype) == 0 || pred->dtype != col->dtype) return -1;
  int64_t words = (col->n + 31) / 32;
  for (int64_t w = 0; w < words; ++w) bitmap[w] = 0;
  for (int64_t r = 0; r < col->n; ++r)
    if (row_pred(*col, *pred, r)) bitmap[r >> 5] |= (uint32_t)1 << (r & 31);
  return 0;
}

void oracle_bitmap_combine(int op, const uint32_t* a, const uint32_t* b, uint32_t* out, int64_t n) {
  int64_t words = (n + 31) / 32;
  for (int64_t w = 0; w < words; ++w) {
    uint32_t v = op == 0 ? (a[w] & b[w]) : (op == 1 ? (a[w] | b[w]) : (a[w] & ~b[w]));
    if (w == words - 1 && (n & 31)) v &= ((uint32_t)1 << (n & 31)) - 1;   // tail bits stay 0
    out[w] = v;
  }
}

int64_t oracle_compact(const uint32_t* bitmap, int64_t n, uint32_t* oids) {
  int64_t m = 0;
  for (int64_t r = 0; r < n; ++r)
    if ((bitmap[r >> 5] >> (r & 31)) & 1) oids[m++] = (uint32_t)r;
  return m;
}

void oracle_gather(const orc_column* col, const uint32_t* oids, int64_t m, void* out) {
  int es = elem_size(col->dtype);
  for (int64_t j = 0; j < m; ++j)
    std::memcpy((char*)out + j * es, (const char*)col->data + (int64_t)oids[j] * es, es);
}

int64_t oracle_group_hash(const orc_column* keys, int nkeys, const uint32_t* oids, int64_t m,
                          int32_t* gids, int64_t* keys_out) {
  if (!keys_valid(keys, nkeys)) return -1;
  std::unordered_map<uint64_t, int32_t> gid_of;
  int64_t G = 0;
  for (int64_t j = 0; j < m; ++j) {
    int64_t r = oids ? (int64_t)oids[j] : j;
    uint64_t k = packed_key(keys, nkeys, r);
    auto it = gid_of.find(k);
    if (it == gid_of.end()) {
      it = gid_of.emplace(k, (int32_t)G).first;
      if (keys_out) keys_out[G] = (int64_t)k;
      ++G;
    }
    gids[j] = it->second;
  }
  return G;
}

int64_t oracle_group_sort(const orc_column* keys, int nkeys, const uint32_t* oids, int64_t m,
                          int32_t* gids, int64_t* keys_out) {
  if (!keys_valid(keys, nkeys)) return -1;
  std::vector<std::pair<uint64_t, int64_t>> kj((size_t)m);
  for (int64_t j = 0; j < m; ++j) {
    int64_t r = oids ? (int64_t)oids[j] : j;
    kj[(size_t)j] = {packed_key(keys, nkeys, r), j};
  }
  std::stable_sort(kj.begin(), kj.end(),
                   [](const std::pair<uint64_t, int64_t>& x, const std::pair<uint64_t, int64_t>& y) { return x.first < y.first; });
  // runs of equal keys; a run's first element has the run's minimum j
  std::vector<std::pair<int64_t, size_t>> runs;   // (min j, start index)
  for (size_t i = 0; i < kj.size(); ++i)
    if (i == 0 || kj[i].first != kj[i - 1].first) runs.push_back({kj[i].second, i});
  std::sort(runs.begin(), runs.end());
  for (size_t g = 0; g < runs.size(); ++g) {
    size_t i = runs[g].second;
    uint64_t k = kj[i].first;
    if (keys_out) keys_out[g] = (int64_t)k;
    for (; i < kj.size() && kj[i].first == k; ++i) gids[kj[i].second] = (int32_t)g;
  }
  return (int64_t)runs.size();
}

// Sorted-input group-by, the paper's first algorithm (§4.1.6):
// "If the input is sorted, we identify group boundaries by having each thread
// compare its value with its successor. Then, a prefix sum operation is used to
// generate dense group IDs."  Step 1: boundary[j] = 1 if key(j) != key(j+1)
// (successor compare; the last row ends a group).  Step 2: exclusive prefix sum
// of the boundaries gives gid[j] = number of group ends before row j.  Sorted
// means non-decreasing packed key (unsigned 64-bit order); returns -2 if a row's
// key is smaller than its predecessor's (nothing else is then guaranteed).
int64_t oracle_group_sorted(const orc_column* keys, int nkeys, const uint32_t* oids, int64_t m,
                            int32_t* gids, int64_t* keys_out) {
  if (!keys_valid(keys, nkeys)) return -1;
  std::vector<uint64_t> k((size_t)m);
  for (int64_t j = 0; j < m; ++j) k[(size_t)j] = packed_key(keys, nkeys, oids ? (int64_t)oids[j] : j);
  for (int64_t j = 1; j < m; ++j)
    if (k[(size_t)j] < k[(size_t)j - 1]) return -2;
  std::vector<int64_t> boundary((size_t)m);
  for (int64_t j = 0; j < m; ++j) boundary[(size_t)j] = (j == m - 1 || k[(size_t)j] != k[(size_t)j + 1]) ? 1 : 0;
  int64_t prefix = 0;                       // exclusive prefix sum of the boundaries
  for (int64_t j = 0; j < m; ++j) {
    gids[j] = (int32_t)prefix;
    if (keys_out && boundary[(size_t)j]) keys_out[prefix] = (int64_t)k[(size_t)j];
    prefix += boundary[(size_t)j];
  }
  return prefix;
}

// Equi-join (§4.1.5): the plain definition — every pair (probe row
// j, build row i) with key(j) == key(i) — evaluated with a std::unordered_map from key
// to the ascending list of build rows.  Pairs in probe order, a probe row's partners in
// ascending build order.  Keys: raw bits masked to the column width (both sides the
// same dtype).  Returns the number of pairs (written only while < out_capacity), or -1.
int64_t oracle_hash_join(const orc_column* build, const orc_column* probe, const uint32_t* oids, int64_t m,
                         uint32_t* out_probe, uint32_t* out_build, int64_t out_capacity) {
  if (!keys_valid(build, 1) || !keys_valid(probe, 1) || build->dtype != probe->dtype) return -1;
  std::unordered_map<uint64_t, std::vector<uint32_t>> rows_of;
  for (int64_t i = 0; i < build->n; ++i) rows_of[packed_key(build, 1, i)].push_back((uint32_t)i);
  int64_t k = 0;
  for (int64_t j = 0; j < m; ++j) {
    const int64_t r = oids ? (int64_t)oids[j] : j;
    auto it = rows_of.find(packed_key(probe, 1, r));
    if (it == rows_of.end()) continue;
    for (uint32_t i : it->second) {
      if (k < out_capacity) {
        out_probe[k] = (uint32_t)r;
        out_build[k] = i;
      }
      ++k;
    }
  }
  return k;
}

int oracle_aggregate(const int32_t* gids, const uint32_t* oids, int64_t m, int64_t G,
                     const orc_column* vals, int nvals, const orc_agg* aggs, int naggs) {
  for (int i = 0; i < naggs; ++i)
    if (!agg_valid(aggs[i], vals, nvals)) return -1;
  std::vector<int64_t> count((size_t)G, 0);
  for (int64_t j = 0; j < m; ++j) count[(size_t)gids[j]]++;
  for (int i = 0; i < naggs; ++i) {
    const orc_agg& g = aggs[i];
    if (g.op == ORC_AGG_COUNT) {
      std::memcpy(g.out, count.data(), (size_t)G * 8);
      continue;
    }
    bool fp = is_f64(vals, g.a);
    if (g.op == ORC_AGG_SUM || g.op == ORC_AGG_AVG) {
      if (fp) {
        std::vector<Neumaier> s((size_t)G);
        for (int64_t j = 0; j < m; ++j) s[(size_t)gids[j]].add(f64_expr(g, vals, oids ? (int64_t)oids[j] : j));
        for (int64_t k = 0; k < G; ++k) {
          double v = s[(size_t)k].value();
          ((double*)g.out)[k] = g.op == ORC_AGG_SUM ? v : v / (double)count[(size_t)k];
        }
      } else {
        std::vector<u128> s((size_t)G, 0);
        for (int64_t j = 0; j < m; ++j) s[(size_t)gids[j]] += int_expr(g, vals, oids ? (int64_t)oids[j] : j);
        for (int64_t k = 0; k < G; ++k) {
          if (g.op == ORC_AGG_SUM) {
            uint64_t lo = (uint64_t)s[(size_t)k];
            int64_t hi = (int64_t)(uint64_t)(s[(size_t)k] >> 64);
            ((uint64_t*)g.out)[2 * k] = lo;
            ((int64_t*)g.out)[2 * k + 1] = hi;
          } else {
            ((double*)g.out)[k] = (double)(i128)s[(size_t)k] / (double)count[(size_t)k];
          }
        }
      }
      continue;
    }
    // MIN / MAX over a plain column
    bool is_min = g.op == ORC_AGG_MIN;
    std::vector<bool> seen((size_t)G, false);
    for (int64_t j = 0; j < m; ++j) {
      int64_t r = oids ? (int64_t)oids[j] : j;
      size_t k = (size_t)gids[j];
      if (fp) {
        double x = f64_value(vals[g.a], r);
        double& o = ((double*)g.out)[k];
        if (!seen[k] || (is_min ? x < o : x > o)) o = x;
      } else {
        int64_t x = int_value(vals[g.a], r);
        int64_t& o = ((int64_t*)g.out)[k];
        if (!seen[k] || (is_min ? x < o : x > o)) o = x;
      }
      seen[k] = true;
    }
  }
  return 0;
}

int64_t oracle_sga(const orc_column* pred_cols, const orc_range* preds, int npreds,
                   const orc_column* key_cols, int nkeys, const orc_column* vals, int nvals,
                   const orc_agg* aggs, int naggs, int order_by_key, int64_t* keys_out,
                   int64_t out_capacity) {
  int64_t n = -1;
  for (int p = 0; p < npreds; ++p) n = pred_cols[p].n;
  for (int k = 0; k < nkeys; ++k) n = key_cols[k].n;
  for (int v = 0; v < nvals; ++v) n = vals[v].n;
  if (n < 0) n = 0;
  for (int i = 0; i < naggs; ++i)
    if (!agg_valid(aggs[i], vals, nvals)) return -1;
  if (nkeys != 0 && !keys_valid(key_cols, nkeys)) return -1;
  // 1. selection: conjunction of range predicates (L429-438)
  int64_t words = (n + 31) / 32;
  std::vector<uint32_t> bitmap((size_t)words, 0), tmp((size_t)words, 0);
  for (int64_t r = 0; r < n; ++r) bitmap[(size_t)(r >> 5)] |= (uint32_t)1 << (r & 31);
  for (int p = 0; p < npreds; ++p) {
    if (oracle_select(&pred_cols[p], &preds[p], tmp.data()) != 0) return -1;
    oracle_bitmap_combine(0, bitmap.data(), tmp.data(), bitmap.data(), n);
  }
  // 2. bitmap -> TIDs (L449-455)
  std::vector<uint32_t> oids((size_t)n);
  int64_t m = oracle_compact(bitmap.data(), n, oids.data());
  // 3. group (L551-561)
  std::vector<int32_t> gids((size_t)m, 0);
  std::vector<int64_t> keys((size_t)(m > 0 ? m : 1), 0);
  int64_t G;
  if (nkeys == 0) G = m > 0 ? 1 : 0;
  else G = oracle_group_hash(key_cols, nkeys, oids.data(), m, gids.data(), keys.data());
  if (G > out_capacity) return -2;
  // 4. aggregate (L562-568) into temporaries, then (optionally) order by key
  std::vector<std::vector<char>> tmp_out((size_t)naggs);
  std::vector<orc_agg> tagg(aggs, aggs + naggs);
  for (int i = 0; i < naggs; ++i) {
    tmp_out[(size_t)i].resize((size_t)(G > 0 ? G : 1) * out_elem_bytes(aggs[i], vals));
    tagg[(size_t)i].out = tmp_out[(size_t)i].data();
  }
  if (oracle_aggregate(gids.data(), oids.data(), m, G, vals, nvals, tagg.data(), naggs) != 0) return -1;
  std::vector<int64_t> order((size_t)G);
  for (int64_t g = 0; g < G; ++g) order[(size_t)g] = g;
  if (order_by_key)
    std::sort(order.begin(), order.end(), [&](int64_t x, int64_t y) { return (uint64_t)keys[(size_t)x] < (uint64_t)keys[(size_t)y]; });
  for (int64_t g = 0; g < G; ++g) {
    if (keys_out) keys_out[g] = keys[(size_t)order[(size_t)g]];
    for (int i = 0; i < naggs; ++i) {
      size_t es = out_elem_bytes(aggs[i], vals);
      std::memcpy((char*)aggs[i].out + (size_t)g * es, tmp_out[(size_t)i].data() + (size_t)order[(size_t)g] * es, es);
    }
  }
  return G;
}

}  // extern "C"
