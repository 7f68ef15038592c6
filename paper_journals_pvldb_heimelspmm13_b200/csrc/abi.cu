// abi.cu — the C ABI (include/ocelot_b200.h): argument validation, planning,
// workspace carving and stream-ordered launches.  The paper's "operator host
// code" (§3.2): check inputs, set up resources, schedule the
// kernels, release everything on error — with caller-owned device memory instead
// of Ocelot's Memory Manager cache (L329-365 §3.3).
#include <math.h>
#include <stdarg.h>
#include <stdio.h>
#include <string.h>

#include <algorithm>

#include <nvtx3/nvToolsExt.h>

#include "launch.cuh"


using namespace ocl;

namespace ocl {
std::atomic<unsigned long long> g_launches{0};
}

struct ocl_ctx {
  cudaEvent_t prof_begin = nullptr, prof_end = nullptr;   // optional: bracket the fused kernel
  cudaEvent_t xchg_begin = nullptr, xchg_end = nullptr;   // optional: bracket exchange + merge (distributed)
  void* comm = nullptr;     // ncclComm_t (ocl_ctx_attach_nccl)
  int rank = 0, nranks = 1;
  int last_kernel = 0;                                     // 0 generic, >0 specialised signature id
  int device;
  int sms;
  int grid;                 // generic grid-stride kernels
  cudaStream_t copy_stream; // host-buffer path
  cudaStream_t comp_stream;
  cudaEvent_t ev_copied[2], ev_consumed[2];
};

namespace {

thread_local char g_err[512] = "";

ocl_status fail(ocl_status s, const char* fmt, ...) {
  va_list ap;
  va_start(ap, fmt);
  vsnprintf(g_err, sizeof(g_err), fmt, ap);
  va_end(ap);
  return s;
}

ocl_status cuda_fail(cudaError_t e, const char* what) {
  return fail(OCL_ERR_CUDA, "%s: %s", what, cudaGetErrorString(e));
}

// NVTX range for the enclosing scope (host-side phase markers; free without a profiler).
struct NvtxRange {
  explicit NvtxRange(const char* name) { nvtxRangePushA(name); }
  ~NvtxRange() { nvtxRangePop(); }
};

#define OCL_CUDA(call, what)                       \
  do {                                             \
    cudaError_t e_ = (call);                       \
    if (e_ != cudaSuccess) return cuda_fail(e_, what); \
  } while (0)

constexpr int64_t kMaxRows = (int64_t)1 << 32;

bool valid_dtype(int32_t d) { return d >= OCL_U8 && d <= OCL_F64; }

size_t align_up(size_t x, size_t a) { return (x + a - 1) / a * a; }

uint64_t next_pow2(uint64_t x) {
  uint64_t c = 1;
  while (c < x) c <<= 1;
  return c;
}

ocl_status check_column(const ocl_column* c, const char* what) {
  if (!c) return fail(OCL_ERR_INVALID_ARG, "%s: NULL column descriptor", what);
  if (!valid_dtype(c->dtype)) return fail(OCL_ERR_INVALID_ARG, "%s: bad dtype %d", what, c->dtype);
  if (c->n < 0 || c->n >= kMaxRows) return fail(OCL_ERR_INVALID_ARG, "%s: n=%lld out of range [0, 2^32)", what, (long long)c->n);
  if (c->n > 0 && !c->data) return fail(OCL_ERR_INVALID_ARG, "%s: NULL data with n > 0", what);
  return OCL_OK;
}

// Normalise a MonetDB range to inclusive bounds lo <= x <= hi (s2).
void normalise_range(const ocl_range& r, int64_t* lo, int64_t* hi, double* flo, double* fhi) {
  *lo = INT64_MIN;
  *hi = INT64_MAX;
  *flo = -INFINITY;
  *fhi = INFINITY;
  if (r.dtype == OCL_F64) {
    if (r.has_lo) {
      if (r.lo_incl) *flo = r.lo_f;
      else if (r.lo_f == INFINITY) { *flo = INFINITY; *fhi = -INFINITY; return; }
      else *flo = nextafter(r.lo_f, INFINITY);
    }
    if (r.has_hi) {
      if (r.hi_incl) *fhi = r.hi_f;
      else if (r.hi_f == -INFINITY) { *flo = INFINITY; *fhi = -INFINITY; return; }
      else *fhi = nextafter(r.hi_f, -INFINITY);
    }
    return;
  }
  if (r.has_lo) {
    if (r.lo_incl) *lo = r.lo_i;
    else if (r.lo_i == INT64_MAX) { *lo = 1; *hi = 0; return; }
    else *lo = r.lo_i + 1;
  }
  if (r.has_hi) {
    if (r.hi_incl) *hi = r.hi_i;
    else if (r.hi_i == INT64_MIN) { *lo = 1; *hi = 0; return; }
    else *hi = r.hi_i - 1;
  }
}

DevCol devcol(const ocl_column& c) { return DevCol{c.data, c.dtype, dtype_width(c.dtype)}; }

bool pair_aligned(const ocl_column& c) {
  return ((uintptr_t)c.data % (uintptr_t)(2 * dtype_width(c.dtype))) == 0;
}

// Plan of one fused / aggregate call.
struct Planned {
  Plan plan;
  FinPlan fin;
  bool values_f64;   // every value expression is fp64
  uint64_t cap;      // table capacity (power of two)
  size_t table_bytes;
  int32_t pbits;     // >= 0: hash-partitioned high-cardinality tier with 2^pbits partitions (partition.cu)
  bool sorted;       // sort-based grouping of sorted input (sorted.cu)
  bool sortgrp;      // tier 6: radix sort, then the sorted path (radix.cu + sorted.cu)
};

ocl_status plan_values(const ocl_column* vals, int32_t nvals, const ocl_agg* aggs, int32_t naggs, Planned* P) {
  Plan& p = P->plan;
  FinPlan& f = P->fin;
  if (naggs < 0 || naggs > kMaxAggs) return fail(OCL_ERR_UNSUPPORTED, "naggs=%d (max %d)", naggs, kMaxAggs);
  if (nvals < 0 || nvals > 16) return fail(OCL_ERR_INVALID_ARG, "nvals=%d", nvals);
  if (naggs > 0 && !aggs) return fail(OCL_ERR_INVALID_ARG, "NULL aggs");
  for (int i = 0; i < nvals; ++i) {
    ocl_status s = check_column(&vals[i], "val_cols");
    if (s) return s;
  }
  struct VKey { int32_t expr, a, b, c, scale; };
  VKey keys[kMaxVals];
  bool need_sum[kMaxVals] = {}, need_min[kMaxVals] = {}, need_max[kMaxVals] = {};
  int vidx[kMaxAggs];
  p.nvals = 0;
  for (int i = 0; i < naggs; ++i) {
    const ocl_agg& g = aggs[i];
    vidx[i] = -1;
    if (g.op < OCL_AGG_COUNT || g.op > OCL_AGG_AVG) return fail(OCL_ERR_INVALID_ARG, "agg %d: bad op %d", i, g.op);
    if (!g.out) return fail(OCL_ERR_INVALID_ARG, "agg %d: NULL out", i);
    if (g.op == OCL_AGG_COUNT) {
      if (g.a >= nvals) return fail(OCL_ERR_INVALID_ARG, "agg %d: COUNT column index %d", i, g.a);
      continue;
    }
    int need = g.expr == OCL_EXPR_COL ? 1 : g.expr == OCL_EXPR_MUL_1MINUS ? 2 : g.expr == OCL_EXPR_MUL_1MINUS_1PLUS ? 3 : -1;
    if (need < 0) return fail(OCL_ERR_INVALID_ARG, "agg %d: bad expr %d", i, g.expr);
    int idx[3] = {g.a, g.b, g.c};
    for (int k = 0; k < need; ++k)
      if (idx[k] < 0 || idx[k] >= nvals) return fail(OCL_ERR_INVALID_ARG, "agg %d: operand %d index %d out of range", i, k, idx[k]);
    bool f64 = vals[g.a].dtype == OCL_F64;
    for (int k = 0; k < need; ++k) {
      if (vals[idx[k]].dtype == OCL_U8) return fail(OCL_ERR_UNSUPPORTED, "agg %d: arithmetic on u8 column", i);
      if ((vals[idx[k]].dtype == OCL_F64) != f64) return fail(OCL_ERR_INVALID_ARG, "agg %d: mixed int/fp64 expression", i);
    }
    if ((g.op == OCL_AGG_MIN || g.op == OCL_AGG_MAX) && g.expr != OCL_EXPR_COL)
      return fail(OCL_ERR_UNSUPPORTED, "agg %d: MIN/MAX over an expression", i);
    if (g.decimal_scale < 0 || g.decimal_scale > 18) return fail(OCL_ERR_INVALID_ARG, "agg %d: decimal_scale %d", i, g.decimal_scale);
    VKey k{g.expr, g.a, need > 1 ? g.b : -1, need > 2 ? g.c : -1, need > 1 ? g.decimal_scale : 0};
    int found = -1;
    for (int v = 0; v < p.nvals; ++v)
      if (!memcmp(&keys[v], &k, sizeof(k))) found = v;
    if (found < 0) {
      if (p.nvals >= kMaxVals) return fail(OCL_ERR_UNSUPPORTED, "more than %d distinct value expressions", kMaxVals);
      found = p.nvals++;
      keys[found] = k;
    }
    vidx[i] = found;
    if (g.op == OCL_AGG_SUM || g.op == OCL_AGG_AVG) need_sum[found] = true;
    if (g.op == OCL_AGG_MIN) need_min[found] = true;
    if (g.op == OCL_AGG_MAX) need_max[found] = true;
  }
  int off = 16;
  P->values_f64 = p.nvals > 0;
  p.has_minmax = 0;
  f.nstates = 0;
  for (int v = 0; v < p.nvals; ++v) {
    DevValue& d = p.vals[v];
    memset(&d, 0, sizeof(d));
    d.expr = keys[v].expr;
    d.a = devcol(vals[keys[v].a]);
    if (keys[v].b >= 0) d.b = devcol(vals[keys[v].b]);
    if (keys[v].c >= 0) d.c = devcol(vals[keys[v].c]);
    d.is_f64 = vals[keys[v].a].dtype == OCL_F64;
    if (!d.is_f64) P->values_f64 = false;
    int64_t S = 1;
    for (int i = 0; i < keys[v].scale; ++i) S *= 10;
    d.S = S;
    d.Sf = (double)S;
    d.off_sum = d.off_min = d.off_max = -1;
    if (need_sum[v]) {
      d.off_sum = off;
      f.states[f.nstates++] = StateDesc{d.is_f64 ? ACC_SUM_F : ACC_SUM_I, off};
      off += d.is_f64 ? 8 : 16;
    }
    if (need_min[v]) {
      d.off_min = off;
      f.states[f.nstates++] = StateDesc{d.is_f64 ? ACC_MIN_F : ACC_MIN_I, off};
      off += 8;
      p.has_minmax = 1;
    }
    if (need_max[v]) {
      d.off_max = off;
      f.states[f.nstates++] = StateDesc{d.is_f64 ? ACC_MAX_F : ACC_MAX_I, off};
      off += 8;
      p.has_minmax = 1;
    }
  }
  // private accumulator record of the register tier: [count u32 | per value: sum lo u64 + hi u32 (int) or
  // f64 | min u64 | max u64], 8-byte fields 8-aligned
  int rec = 4;
  for (int v = 0; v < p.nvals; ++v) {
    DevValue& d = p.vals[v];
    d.po_sum = d.po_hi = d.po_min = d.po_max = -1;
    if (need_sum[v]) {
      rec = (int)align_up((size_t)rec, 8);
      d.po_sum = rec;
      rec += 8;
      if (!d.is_f64 && d.expr != OCL_EXPR_COL) { d.po_hi = rec; rec += 4; }   // products: 96-bit
    }
    if (need_min[v]) { rec = (int)align_up((size_t)rec, 8); d.po_min = rec; rec += 8; }
    if (need_max[v]) { rec = (int)align_up((size_t)rec, 8); d.po_max = rec; rec += 8; }
  }
  p.priv_rec = (int)align_up((size_t)rec, 8);
  {   // CTA-table entry layout: [~key u64][count u32] per value [lo16 sum][hi16 sum][min][max]
    int co = 12;
    for (int v = 0; v < p.nvals; ++v) {
      DevValue& d = p.vals[v];
      d.co_lo = d.co_hi = d.co_min = d.co_max = -1;
      if (d.off_sum >= 0) { d.co_lo = co; d.co_hi = co + 4; co += 8; }
      if (d.off_min >= 0) { d.co_min = co; co += 4; }
      if (d.off_max >= 0) { d.co_max = co; co += 4; }
    }
    p.cta_stride = (int)align_up((size_t)co, 8);
  }
  // distinct operand columns (static shapes load each once) and per-value indices
  p.ncols = 0;
  auto col_index = [&](const DevCol& c) -> int {
    for (int i = 0; i < p.ncols; ++i)
      if (p.vcols[i].ptr == c.ptr && p.vcols[i].dtype == c.dtype) return i;
    if (p.ncols == kMaxCols) return -1;
    p.vcols[p.ncols] = c;
    return p.ncols++;
  };
  for (int v = 0; v < p.nvals; ++v) {
    DevValue& d = p.vals[v];
    d.ia = col_index(d.a);
    d.ib = d.expr >= OCL_EXPR_MUL_1MINUS ? col_index(d.b) : 0;
    d.ic = d.expr >= OCL_EXPR_MUL_1MINUS_1PLUS ? col_index(d.c) : 0;
  }
  int stride = (int)align_up((size_t)off, 16);
  if (stride <= 32) stride = 32;
  else if (stride <= 64) stride = 64;
  else stride = (int)align_up((size_t)stride, 32);
  p.stride = stride;
  f.stride = stride;
  f.naggs = naggs;
  for (int i = 0; i < naggs; ++i) {
    const ocl_agg& g = aggs[i];
    OutAgg& o = f.aggs[i];
    o.op = g.op;
    o.out = g.out;
    if (g.op == OCL_AGG_COUNT) { o.kind = -1; o.off = 8; o.is_f64 = 0; continue; }
    const DevValue& d = p.vals[vidx[i]];
    o.is_f64 = d.is_f64;
    if (g.op == OCL_AGG_SUM || g.op == OCL_AGG_AVG) { o.off = d.off_sum; o.kind = d.is_f64 ? ACC_SUM_F : ACC_SUM_I; }
    else if (g.op == OCL_AGG_MIN) { o.off = d.off_min; o.kind = d.is_f64 ? ACC_MIN_F : ACC_MIN_I; }
    else { o.off = d.off_max; o.kind = d.is_f64 ? ACC_MAX_F : ACC_MAX_I; }
  }
  return OCL_OK;
}

ocl_status plan_keys(const ocl_column* key_cols, int32_t nkeys, Plan& p) {
  if (nkeys < 0 || nkeys > kMaxKeys) return fail(OCL_ERR_INVALID_ARG, "nkeys=%d (0..2)", nkeys);
  if (nkeys > 0 && !key_cols) return fail(OCL_ERR_INVALID_ARG, "NULL key_cols");
  int bits = 0;
  for (int i = 0; i < nkeys; ++i) {
    ocl_status s = check_column(&key_cols[i], "key_cols");
    if (s) return s;
    if (key_cols[i].dtype == OCL_F64) return fail(OCL_ERR_INVALID_ARG, "key column %d is f64", i);
    bits += 8 * dtype_width(key_cols[i].dtype);
  }
  if (bits > 64) return fail(OCL_ERR_INVALID_ARG, "packed key width %d bits > 64", bits);
  p.nkeys = nkeys;
  int shift = 0;
  for (int i = nkeys - 1; i >= 0; --i) {   // key = a << width(b) | b
    int w = 8 * dtype_width(key_cols[i].dtype);
    p.keys[i].col = devcol(key_cols[i]);
    p.keys[i].shift = shift;
    p.keys[i].mask = w == 64 ? ~0ULL : ((1ULL << w) - 1);
    shift += w;
  }
  return OCL_OK;
}

ocl_status plan_preds(const ocl_column* pred_cols, const ocl_range* preds, int32_t npreds, Plan& p) {
  if (npreds < 0 || npreds > kMaxPreds) return fail(OCL_ERR_UNSUPPORTED, "npreds=%d (max %d)", npreds, kMaxPreds);
  if (npreds > 0 && (!pred_cols || !preds)) return fail(OCL_ERR_INVALID_ARG, "NULL pred_cols/preds");
  p.npreds = npreds;
  for (int i = 0; i < npreds; ++i) {
    ocl_status s = check_column(&pred_cols[i], "pred_cols");
    if (s) return s;
    if (preds[i].dtype != pred_cols[i].dtype) return fail(OCL_ERR_INVALID_ARG, "pred %d: range dtype != column dtype", i);
    DevPred& d = p.preds[i];
    d.col = devcol(pred_cols[i]);
    d.is_f64 = pred_cols[i].dtype == OCL_F64;
    d.anti = preds[i].anti ? 1 : 0;
    normalise_range(preds[i], &d.lo, &d.hi, &d.flo, &d.fhi);
    if (d.lo > d.hi || d.lo > INT32_MAX || d.hi < INT32_MIN) { d.lo32 = 1; d.hi32 = 0; }   // empty range
    else {
      d.lo32 = (int32_t)std::max<int64_t>(d.lo, INT32_MIN);
      d.hi32 = (int32_t)std::min<int64_t>(d.hi, INT32_MAX);
    }
  }
  return OCL_OK;
}

// Shared-memory budget of one register-tier CTA (private records + mid-G table).
constexpr size_t kRegTierSmem = 200 * 1024;
// Auto selection of the hash-partitioned tier: above 1024 expected groups
// it beats the fused kernel's shared-memory CTA table (C5, 2^28 rows, sel 100 %: 2048
// groups 10.6 -> 8.8 ms, 4096 groups 14.7 -> 8.5 ms; at 1024 the fused kernel wins).
constexpr int64_t kPartMinGroups = 1024;
constexpr int64_t kPartMinRows = 1 << 20;

// Tier selection: 0 auto; 1 register tier (private slots + HBM);
// 2 HBM-only kernel; 3 register tier with the dynamic (unspecialised) shape;
// 4 register tier with the CTA shared-memory table forced on.
int fused_mode(const ocl_sga_args* a) {
  if (a->tier == 2) return 2;
  if (a->tier == 3) return 1;
  if (a->tier == 4) return 3;
  return 0;
}

// CTA shared-table capacity for the register tier (0 = none).  Eligible plans:
// every value an integer column (its fast path is int32, the table's field width).
int32_t plan_smem_cap(const ocl_sga_args* a, const Plan& p) {
  if (a->tier == 1 || a->tier == 2 || a->tier == 3) return 0;
  for (int v = 0; v < p.nvals; ++v)
    if (p.vals[v].is_f64 || p.vals[v].expr != OCL_EXPR_COL) return 0;
  const size_t priv = (size_t)reg_tier_slots() * p.priv_rec * 256;
  if (priv >= kRegTierSmem) return 0;
  const uint64_t fit = next_pow2((kRegTierSmem - priv) / (size_t)p.cta_stride + 1) / 2;   // largest pow2 that fits
  if (a->tier == 4) return (int32_t)std::min<uint64_t>(fit, 1u << 14);
  if (a->expected_groups <= reg_tier_slots()) return 0;
  const uint64_t cap = next_pow2((uint64_t)std::max<int64_t>(2 * a->expected_groups, 64));
  return cap <= fit ? (int32_t)cap : 0;     // too many groups for shared memory: HBM table
}

ocl_status plan_sga(const ocl_sga_args* a, Planned* P, bool need_outputs = true) {
  if (!a) return fail(OCL_ERR_INVALID_ARG, "NULL args");
  memset(P, 0, sizeof(*P));
  Plan& p = P->plan;
  ocl_status s;
  if ((s = plan_preds(a->pred_cols, a->preds, a->npreds, p))) return s;
  if ((s = plan_keys(a->key_cols, a->nkeys, p))) return s;
  if ((s = plan_values(a->val_cols, a->nvals, a->aggs, a->naggs, P))) return s;
  int64_t n = -1;
  bool aligned = true;
  auto see = [&](const ocl_column& c) -> bool {
    if (n >= 0 && c.n != n) return false;
    n = c.n;
    aligned = aligned && pair_aligned(c);
    return true;
  };
  for (int i = 0; i < a->npreds; ++i)
    if (!see(a->pred_cols[i])) return fail(OCL_ERR_INVALID_ARG, "columns differ in length");
  for (int i = 0; i < a->nkeys; ++i)
    if (!see(a->key_cols[i])) return fail(OCL_ERR_INVALID_ARG, "columns differ in length");
  for (int i = 0; i < a->nvals; ++i)
    if (!see(a->val_cols[i])) return fail(OCL_ERR_INVALID_ARG, "columns differ in length");
  p.n = n < 0 ? 0 : n;
  p.vec_ok = aligned ? 1 : 0;
  if (need_outputs && !a->ngroups_out) return fail(OCL_ERR_INVALID_ARG, "NULL ngroups_out");
  if (a->out_capacity < 0) return fail(OCL_ERR_INVALID_ARG, "out_capacity < 0");
  int64_t expected = a->expected_groups > 0 ? a->expected_groups : 1;
  if (expected > ((int64_t)1 << 40)) return fail(OCL_ERR_INVALID_ARG, "expected_groups too large");
  P->cap = next_pow2((uint64_t)std::max<int64_t>(2 * expected, 16));
  p.mask = P->cap - 1;
  P->table_bytes = align_up((P->cap + 1) * (size_t)p.stride, 256);
  p.status = a->dev_status;
  p.bitmap_out = a->bitmap_out;
  p.expected = expected;
  p.smem_cap = plan_smem_cap(a, p);
  p.miss_agg = a->expected_groups > reg_tier_slots() ? 1 : 0;
  // High-cardinality tier: more groups than the shared-memory tiers hold, integer
  // column values, enough rows to amortise its five launches (tier 5 forces it).
  P->pbits = -1;
  const bool many = a->tier == 0 && a->expected_groups > kPartMinGroups && p.n >= kPartMinRows && !spec_takes(p);
  if ((a->tier == 5 || many) && part_eligible(p)) P->pbits = part_bits_for(a->expected_groups, p.n);
  P->sorted = a->key_sorted != 0;
  P->sortgrp = a->tier == 6;
  if (P->sortgrp) {
    if (a->key_sorted) return fail(OCL_ERR_INVALID_ARG, "tier 6 sorts the input itself: key_sorted must be 0");
    if (a->npreds != 0 || a->nkeys == 0) return fail(OCL_ERR_UNSUPPORTED, "tier 6: no predicate, >= 1 key column");
    if (p.ncols > 1 || (p.ncols == 1 && p.vcols[0].width != 8))
      return fail(OCL_ERR_UNSUPPORTED, "tier 6: at most one distinct 8-byte value column");
    P->pbits = -1;
    P->table_bytes = 0;
  }
  if (P->sorted) {
    if (a->tier != 0) return fail(OCL_ERR_INVALID_ARG, "key_sorted needs tier 0");
    if (a->nkeys == 0) return fail(OCL_ERR_INVALID_ARG, "key_sorted needs a key column");
    P->pbits = -1;
    P->table_bytes = 0;
  }
  FinPlan& f = P->fin;
  f.order_by_key = a->order_by_key ? 1 : 0;
  f.keys_out = a->keys_out;
  f.ngroups_out = a->ngroups_out;
  f.out_capacity = a->out_capacity;
  f.status = a->dev_status;
  if (a->order_by_key && !P->sorted && !P->sortgrp && !sorted_emit_supported(P->cap))
    return fail(OCL_ERR_UNSUPPORTED, "order_by_key needs expected_groups <= 2047 (table of %llu slots)", (unsigned long long)P->cap);
  return OCL_OK;
}


// table + finalize workspace of a fused call
// tier 6 plan over the sorted copies: one packed i64 key column, the value column re-pointed
Plan sortgrp_plan(const Plan& p0, const uint64_t* skeys, const uint64_t* svals) {
  Plan q = p0;
  q.nkeys = 1;
  q.keys[0].col = DevCol{skeys, OCL_I64, 8};
  q.keys[0].shift = 0;
  q.keys[0].mask = ~0ULL;
  const void* v0 = p0.ncols ? p0.vcols[0].ptr : nullptr;
  auto remap = [&](DevCol& c) { if (v0 && c.ptr == v0) c.ptr = svals; };
  for (int i = 0; i < q.ncols; ++i) remap(q.vcols[i]);
  for (int v = 0; v < q.nvals; ++v) {
    remap(q.vals[v].a);
    remap(q.vals[v].b);
    remap(q.vals[v].c);
  }
  q.vec_ok = 1;
  return q;
}

size_t sga_ws_bytes(ocl_ctx* ctx, const Planned& P) {
  if (P.sortgrp) {
    const int64_t n = P.plan.n;
    return align_up((size_t)n * 8, 256) * 2 + radix_ws_bytes(n, P.plan.ncols > 0, false) + sorted_ws_bytes(P.plan);
  }
  if (P.sorted) return sorted_ws_bytes(P.plan);
  return P.table_bytes + align_up(emit_ws_bytes(ctx->grid), 256) +
         (P.pbits >= 0 ? part_ws_bytes(P.plan, P.pbits, ctx->sms) : 0);
}

// Run the fused pass into a zeroed table carved from ws; returns the emit workspace.
// ea / count_out / cap: the emission the caller wants; the hash-partitioned tier performs it
// itself (*emitted = true), otherwise the caller emits from the table.
ocl_status run_fused(ocl_ctx* ctx, const ocl_sga_args* a, Planned& P, void* ws, size_t ws_bytes, cudaStream_t s,
                     void** emit_ws, const EmitArgs* ea = nullptr, int64_t* count_out = nullptr, int64_t cap = 0,
                     bool* emitted = nullptr) {
  if (emitted) *emitted = false;
  size_t need = sga_ws_bytes(ctx, P);
  if (ws_bytes < need || (!ws && need)) return fail(OCL_ERR_CAPACITY, "workspace %zu B < required %zu B", ws_bytes, need);
  P.plan.table = (uint8_t*)ws;
  *emit_ws = (uint8_t*)ws + P.table_bytes;
  if (P.pbits < 0 || P.plan.n == 0)      // the partitioned tier zeroes (only what it uses) itself
    OCL_CUDA(cudaMemsetAsync(ws, 0, P.table_bytes, s), "table init");
  if (a->dev_status) OCL_CUDA(cudaMemsetAsync(a->dev_status, 0, sizeof(int32_t), s), "status init");
  if (P.plan.n > 0) {
    if (ctx->prof_begin) OCL_CUDA(cudaEventRecord(ctx->prof_begin, s), "profile event");
    int kind = 0;
    if (P.pbits >= 0) {
      void* pws = (uint8_t*)ws + P.table_bytes + align_up(emit_ws_bytes(ctx->grid), 256);
      OCL_CUDA(launch_partitioned(P.plan, P.pbits, pws, ctx->sms, s, &kind, ea, count_out, cap, emitted),
               "partitioned aggregation launch");
    } else {
      OCL_CUDA(launch_fused(P.plan, fused_mode(a), P.values_f64, ctx->sms, s, &kind), "fused kernel launch");
    }
    ctx->last_kernel = kind;
    if (ctx->prof_end) OCL_CUDA(cudaEventRecord(ctx->prof_end, s), "profile event");
  }
  return OCL_OK;
}

// Sort-based grouping (key_sorted = 1: the sorted path; tier 6: radix sort, then the sorted
// path).  partial_out != NULL: partial rows for the multi-GPU merge instead of final outputs,
// count -> *count_out (capacity cap).
ocl_status run_sortpath(ocl_ctx* ctx, const ocl_sga_args* args, const Planned& P, void* ws, size_t ws_bytes,
                        cudaStream_t st, uint8_t* partial_out, int64_t cap, int64_t* count_out) {
  size_t need = sga_ws_bytes(ctx, P);
  if (ws_bytes < need || !ws) return fail(OCL_ERR_CAPACITY, "workspace %zu B < required %zu B", ws_bytes, need);
  if (args->dev_status) OCL_CUDA(cudaMemsetAsync(args->dev_status, 0, sizeof(int32_t), st), "status init");
  if (ctx->prof_begin) OCL_CUDA(cudaEventRecord(ctx->prof_begin, st), "profile event");
  int kind = 0;
  if (P.sortgrp) {                // tier 6: radix sort then the sorted path
    const int64_t n = P.plan.n;
    uint8_t* w = (uint8_t*)ws;
    uint64_t* skeys = (uint64_t*)w;
    uint64_t* svals = (uint64_t*)(w + align_up((size_t)n * 8, 256));
    void* rws = w + 2 * align_up((size_t)n * 8, 256);
    void* sws = (uint8_t*)rws + radix_ws_bytes(n, P.plan.ncols > 0, false);
    if (n == 0) {
      OCL_CUDA(cudaMemsetAsync(count_out, 0, 8, st), "group count");
    } else {
      OCL_CUDA(launch_radix(P.plan, P.plan.ncols ? (const uint64_t*)P.plan.vcols[0].ptr : nullptr, skeys,
                            P.plan.ncols ? svals : nullptr, nullptr, rws, ctx->sms, st), "radix sort");
      OCL_CUDA(launch_sorted(sortgrp_plan(P.plan, skeys, svals), P.fin, P.values_f64, sws, args->dev_status,
                             count_out, cap, ctx->sms, st, &kind, partial_out), "sorted group-by");
      ctx->last_kernel = 50 + (kind - 40);
    }
  } else {                        // sorted input: no table, outputs written by the kernels
    OCL_CUDA(launch_sorted(P.plan, P.fin, P.values_f64, ws, args->dev_status, count_out, cap, ctx->sms, st, &kind,
                           partial_out), "sorted group-by launch");
    ctx->last_kernel = kind;
  }
  if (ctx->prof_end) OCL_CUDA(cudaEventRecord(ctx->prof_end, st), "profile event");
  return OCL_OK;
}

// Local fused pass that emits partial rows (ocl_sga_partial; the local step of a distributed
// call): count -> *count_out, rows -> partial_out (capacity cap); overflow -> args->dev_status.
ocl_status local_partial(ocl_ctx* ctx, const ocl_sga_args* args, Planned& P, void* ws, size_t ws_bytes,
                         cudaStream_t st, uint8_t* partial_out, int64_t cap, int64_t* count_out) {
  if (P.sorted || P.sortgrp) return run_sortpath(ctx, args, P, ws, ws_bytes, st, partial_out, cap, count_out);
  void* ews = nullptr;
  EmitArgs ea;
  memset(&ea, 0, sizeof(ea));
  ea.kind = EMIT_PARTIAL;
  ea.out_capacity = cap;
  ea.partial_out = partial_out;
  ea.status = args->dev_status;
  bool emitted = false;
  ocl_status s = run_fused(ctx, args, P, ws, ws_bytes, st, &ews, &ea, count_out, cap, &emitted);
  if (s) return s;
  if (!emitted)
    OCL_CUDA(launch_emit(P.plan.table, P.cap, P.plan.stride, ea, count_out, cap, args->dev_status, false, ews,
                         ctx->grid, st), "partial export");
  return OCL_OK;
}

// ---------------------------------------------------------------- distributed calls (distributed.cu)
// Workspace of a distributed call: [local step (size `local`)] then the exchange region:
// header (W int64: row count(s) + the local partial's status word), all ranks' headers,
// the local partial table, the all-to-all send blocks, the receive buffer (P parts), the
// per-part row counts, the merge table and its emit scratch.
struct DistLayout {
  int mode, P, W;
  int64_t part_cap;   // partial rows of this rank (= out_capacity)
  int64_t block;      // rows per destination block (all-to-all)
  int64_t recv_cap;   // rows per received part
  uint64_t mcap;      // merge table slots
  size_t rb;          // partial row bytes
  size_t off_hdr, off_hdr_all, off_pcount, off_part, off_send, off_recv, off_counts, off_mtable, off_mews, total;
};

ocl_status dist_layout(ocl_ctx* ctx, const ocl_sga_args* a, const Planned& P, size_t local, DistLayout* L) {
  if (!ctx->comm)
    return fail(OCL_ERR_INVALID_ARG, "distributed = %d but ctx has no NCCL communicator (ocl_ctx_attach_nccl)",
                a->distributed);
  if (a->distributed != 1 && a->distributed != 2)
    return fail(OCL_ERR_INVALID_ARG, "distributed = %d (0 local, 1 allgather, 2 all-to-all)", a->distributed);
  memset(L, 0, sizeof(*L));
  L->mode = a->distributed;
  L->P = ctx->nranks;
  L->W = L->mode == 1 ? 2 : L->P + 1;
  L->rb = (size_t)P.plan.stride;
  L->part_cap = std::max<int64_t>(a->out_capacity, 1);
  L->block = L->mode == 1 ? L->part_cap : (L->part_cap * 5 / 4 + L->P - 1) / L->P + 64;
  L->recv_cap = L->block;
  const int64_t gmax = std::min<int64_t>((int64_t)L->P * L->recv_cap, std::max<int64_t>(a->out_capacity, 1));
  L->mcap = next_pow2((uint64_t)std::max<int64_t>(2 * gmax, 16));
  if (a->order_by_key && !sorted_emit_supported(L->mcap))
    return fail(OCL_ERR_UNSUPPORTED, "order_by_key on a distributed call needs out_capacity <= 1023 (merge table of %llu slots)",
                (unsigned long long)L->mcap);
  size_t o = align_up(local, 256);
  L->off_hdr = o;
  o += align_up((size_t)L->W * 8, 256);
  L->off_hdr_all = o;
  o += align_up((size_t)L->P * L->W * 8, 256);
  L->off_pcount = o;
  o += 256;
  L->off_part = o;
  o += align_up((size_t)L->part_cap * L->rb, 256);
  L->off_send = o;
  if (L->mode == 2) o += align_up((size_t)L->P * L->block * L->rb, 256);
  L->off_recv = o;
  o += align_up((size_t)L->P * L->recv_cap * L->rb, 256);
  L->off_counts = o;
  o += align_up((size_t)L->P * 8, 256);
  L->off_mtable = o;
  o += align_up((L->mcap + 1) * L->rb, 256);
  L->off_mews = o;
  o += align_up(emit_ws_bytes(ctx->grid), 256);
  L->total = o;
  return OCL_OK;
}

// Exchange this rank's partial table (already in the region, its row count in the header
// (allgather) or at off_pcount (all-to-all)) and merge the received parts into fin's outputs.
ocl_status dist_exchange_merge(ocl_ctx* ctx, const ocl_sga_args* a, const DistLayout& L, uint8_t* ws,
                               const FinPlan& fin, int64_t* ngroups_out, int32_t* status, cudaStream_t st) {
  int64_t* hdr = (int64_t*)(ws + L.off_hdr);
  int64_t* hdr_all = (int64_t*)(ws + L.off_hdr_all);
  uint8_t* part = ws + L.off_part;
  uint8_t* recv = ws + L.off_recv;
  int64_t* counts = (int64_t*)(ws + L.off_counts);
  uint8_t* mtable = ws + L.off_mtable;
  char err[256];
  if (ctx->xchg_begin) OCL_CUDA(cudaEventRecord(ctx->xchg_begin, st), "phase event");
  if (L.mode == 1) {
    NvtxRange nv("ocl:allgather");
    if (nccl_allgather2(hdr, hdr_all, (size_t)L.W * 8, part, recv, (size_t)L.part_cap * L.rb, ctx->comm, st, err,
                        sizeof(err)))
      return fail(OCL_ERR_NCCL, "%s", err);
  } else {
    NvtxRange nv("ocl:alltoall");
    uint8_t* send = ws + L.off_send;
    OCL_CUDA(launch_route_blocks(part, (const int64_t*)(ws + L.off_pcount), L.part_cap, (int32_t)L.rb, L.P, L.block,
                                 send, hdr, ctx->sms, st), "route partial rows");
    if (nccl_alltoall_blocks(hdr, hdr_all, (size_t)L.W * 8, send, recv, (size_t)L.block * L.rb, L.P, ctx->comm, st,
                             err, sizeof(err)))
      return fail(OCL_ERR_NCCL, "%s", err);
  }
  NvtxRange nv("ocl:merge");
  const int64_t hcap = L.mode == 1 ? L.part_cap : L.block;
  OCL_CUDA(launch_dist_headers(hdr_all, L.P, L.W, L.mode == 1 ? 0 : ctx->rank, hcap, counts, status, 0, nullptr, st),
           "exchange headers");
  OCL_CUDA(cudaMemsetAsync(mtable, 0, align_up((L.mcap + 1) * L.rb, 256), st), "merge table init");
  OCL_CUDA(launch_merge_partials(recv, L.P, L.recv_cap, counts, fin, mtable, L.mcap - 1, status, ctx->grid, st),
           "merge");
  EmitArgs ea;
  memset(&ea, 0, sizeof(ea));
  ea.kind = EMIT_FINAL;
  ea.fin = fin;
  OCL_CUDA(launch_emit(mtable, L.mcap, (int32_t)L.rb, ea, ngroups_out, a->out_capacity, status, a->order_by_key != 0,
                       ws + L.off_mews, ctx->grid, st), "merge finalize");
  OCL_CUDA(launch_dist_headers(hdr_all, L.P, L.W, 0, hcap, nullptr, nullptr, 1, ngroups_out, st), "overflow report");
  if (ctx->xchg_end) OCL_CUDA(cudaEventRecord(ctx->xchg_end, st), "phase event");
  return OCL_OK;
}

// Local step of a distributed device call: the caller's plan with its own status word (the
// header's, so a local overflow reaches every rank) and no ORDER BY (partial rows).
ocl_status dist_local_plan(ocl_ctx* ctx, const ocl_sga_args* args, ocl_sga_args* la, Planned* PL, size_t* local) {
  *la = *args;
  la->distributed = 0;
  la->order_by_key = 0;
  la->dev_status = nullptr;
  ocl_status s = plan_sga(la, PL, false);
  if (s) return s;
  *local = sga_ws_bytes(ctx, *PL);
  return OCL_OK;
}

ocl_status dist_ws_bytes(ocl_ctx* ctx, const ocl_sga_args* args, const Planned& P, size_t* bytes) {
  ocl_sga_args la;
  Planned PL;
  size_t local = 0;
  ocl_status s = dist_local_plan(ctx, args, &la, &PL, &local);
  if (s) return s;
  DistLayout L;
  if ((s = dist_layout(ctx, args, P, local, &L))) return s;
  *bytes = L.total;
  return OCL_OK;
}

ocl_status run_distributed(ocl_ctx* ctx, const ocl_sga_args* args, const Planned& P, void* ws, size_t ws_bytes,
                           cudaStream_t st) {
  ocl_sga_args la;
  Planned PL;
  size_t local = 0;
  ocl_status s = dist_local_plan(ctx, args, &la, &PL, &local);
  if (s) return s;
  DistLayout L;
  if ((s = dist_layout(ctx, args, P, local, &L))) return s;
  if (!ws || ws_bytes < L.total) return fail(OCL_ERR_CAPACITY, "workspace %zu B < required %zu B", ws_bytes, L.total);
  uint8_t* w = (uint8_t*)ws;
  int64_t* hdr = (int64_t*)(w + L.off_hdr);
  la.dev_status = (int32_t*)&hdr[L.W - 1];
  if ((s = plan_sga(&la, &PL, false))) return s;
  OCL_CUDA(cudaMemsetAsync(hdr, 0, (size_t)L.W * 8, st), "header init");
  if (args->dev_status) OCL_CUDA(cudaMemsetAsync(args->dev_status, 0, 4, st), "status init");
  {
    NvtxRange nv("ocl:select+aggregate (local shard)");
    if ((s = local_partial(ctx, &la, PL, ws, local, st, w + L.off_part, L.part_cap,
                           L.mode == 1 ? hdr : (int64_t*)(w + L.off_pcount))))
      return s;
  }
  return dist_exchange_merge(ctx, args, L, w, P.fin, args->ngroups_out, args->dev_status, st);
}

// Restart ladder of ocl_select_group_aggregate_sync: expected_groups x 4 per step, capped at
// max(out_capacity, expected_groups).  Its workspace is the largest over the ladder.
int sync_ladder(const ocl_sga_args* a, int64_t* egs, int maxn) {
  int64_t eg = std::max<int64_t>(a->expected_groups, 1);
  const int64_t top = std::max<int64_t>(a->out_capacity, eg);
  int n = 0;
  egs[n++] = eg;
  while (eg < top && n < maxn) {
    eg = std::min<int64_t>(eg * 4, top);
    egs[n++] = eg;
  }
  return n;
}

}  // namespace

// ======================================================================== ABI
extern "C" {

int32_t ocl_version(void) { return 1; }

uint64_t ocl_launch_count(void) { return g_launches.load(); }

const char* ocl_ctx_last_kernel(ocl_ctx* ctx) { return ctx ? fused_kernel_name(ctx->last_kernel) : ""; }

ocl_status ocl_ctx_set_kernel_events(ocl_ctx* ctx, void* begin_event, void* end_event) {
  if (!ctx) return fail(OCL_ERR_INVALID_ARG, "NULL ctx");
  ctx->prof_begin = (cudaEvent_t)begin_event;
  ctx->prof_end = (cudaEvent_t)end_event;
  return OCL_OK;
}

ocl_status ocl_ctx_set_phase_events(ocl_ctx* ctx, int32_t phase, void* begin_event, void* end_event) {
  if (!ctx) return fail(OCL_ERR_INVALID_ARG, "NULL ctx");
  if (phase == 0) return ocl_ctx_set_kernel_events(ctx, begin_event, end_event);
  if (phase != 1) return fail(OCL_ERR_INVALID_ARG, "phase %d (0 fused kernel, 1 exchange + merge)", phase);
  ctx->xchg_begin = (cudaEvent_t)begin_event;
  ctx->xchg_end = (cudaEvent_t)end_event;
  return OCL_OK;
}

ocl_status ocl_nccl_unique_id(void* id_out) {
  if (!id_out) return fail(OCL_ERR_INVALID_ARG, "NULL id_out");
  char err[256];
  if (nccl_unique_id(id_out, err, sizeof(err))) return fail(OCL_ERR_NCCL, "%s", err);
  return OCL_OK;
}

ocl_status ocl_ctx_attach_nccl(ocl_ctx* ctx, const void* nccl_unique_id, int32_t rank, int32_t nranks) {
  if (!ctx || !nccl_unique_id) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/unique id");
  if (nranks < 1 || rank < 0 || rank >= nranks || nranks > 1024)
    return fail(OCL_ERR_INVALID_ARG, "rank %d of %d", rank, nranks);
  NvtxRange nv("ocl:nccl_init");
  OCL_CUDA(cudaSetDevice(ctx->device), "cudaSetDevice");
  char err[256];
  void* comm = nullptr;
  if (nccl_comm_init(&comm, nccl_unique_id, rank, nranks, err, sizeof(err))) return fail(OCL_ERR_NCCL, "%s", err);
  nccl_comm_destroy(ctx->comm);
  ctx->comm = comm;
  ctx->rank = rank;
  ctx->nranks = nranks;
  return OCL_OK;
}

ocl_status ocl_ctx_nccl_rank(ocl_ctx* ctx, int32_t* rank, int32_t* nranks) {
  if (!ctx || !rank || !nranks) return fail(OCL_ERR_INVALID_ARG, "NULL argument");
  *rank = ctx->rank;
  *nranks = ctx->nranks;
  return OCL_OK;
}

const char* ocl_last_error(void) { return g_err; }

const char* ocl_status_string(ocl_status s) {
  switch (s) {
    case OCL_OK: return "OCL_OK";
    case OCL_ERR_INVALID_ARG: return "OCL_ERR_INVALID_ARG";
    case OCL_ERR_UNSUPPORTED: return "OCL_ERR_UNSUPPORTED";
    case OCL_ERR_CAPACITY: return "OCL_ERR_CAPACITY";
    case OCL_ERR_OUT_OF_MEMORY: return "OCL_ERR_OUT_OF_MEMORY";
    case OCL_ERR_CUDA: return "OCL_ERR_CUDA";
    case OCL_ERR_NCCL: return "OCL_ERR_NCCL";
  }
  return "OCL_ERR_UNKNOWN";
}

ocl_status ocl_ctx_create(int device, ocl_ctx** out) {
  if (!out) return fail(OCL_ERR_INVALID_ARG, "NULL out");
  *out = nullptr;
  int ndev = 0;
  OCL_CUDA(cudaGetDeviceCount(&ndev), "cudaGetDeviceCount");
  if (device < 0 || device >= ndev) return fail(OCL_ERR_INVALID_ARG, "device %d of %d", device, ndev);
  cudaDeviceProp prop;
  OCL_CUDA(cudaGetDeviceProperties(&prop, device), "cudaGetDeviceProperties");
  if (prop.major != 10 || prop.minor != 0)
    return fail(OCL_ERR_UNSUPPORTED, "device %d is sm_%d%d; libocelot_b200 is built for sm_100a (B200) only", device,
                prop.major, prop.minor);
  OCL_CUDA(cudaSetDevice(device), "cudaSetDevice");
  ocl_ctx* c = new ocl_ctx();
  c->device = device;
  c->sms = prop.multiProcessorCount;
  c->grid = c->sms * 8;
  OCL_CUDA(cudaStreamCreateWithFlags(&c->copy_stream, cudaStreamNonBlocking), "stream create");
  OCL_CUDA(cudaStreamCreateWithFlags(&c->comp_stream, cudaStreamNonBlocking), "stream create");
  for (int i = 0; i < 2; ++i) {
    OCL_CUDA(cudaEventCreateWithFlags(&c->ev_copied[i], cudaEventDisableTiming), "event create");
    OCL_CUDA(cudaEventCreateWithFlags(&c->ev_consumed[i], cudaEventDisableTiming), "event create");
  }
  *out = c;
  return OCL_OK;
}

ocl_status ocl_ctx_destroy(ocl_ctx* ctx) {
  if (!ctx) return OCL_OK;
  nccl_comm_destroy(ctx->comm);
  cudaStreamDestroy(ctx->copy_stream);
  cudaStreamDestroy(ctx->comp_stream);
  for (int i = 0; i < 2; ++i) {
    cudaEventDestroy(ctx->ev_copied[i]);
    cudaEventDestroy(ctx->ev_consumed[i]);
  }
  delete ctx;
  return OCL_OK;
}

// ---------------------------------------------------------------- a1 / A2
ocl_status ocl_select_bitmap(ocl_ctx* ctx, const ocl_column* col, const ocl_range* pred, uint32_t* bitmap_out,
                             void* stream) {
  if (!ctx || !pred) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/pred");
  ocl_status s = check_column(col, "col");
  if (s) return s;
  if (pred->dtype != col->dtype) return fail(OCL_ERR_INVALID_ARG, "range dtype %d != column dtype %d", pred->dtype, col->dtype);
  if (col->n > 0 && !bitmap_out) return fail(OCL_ERR_INVALID_ARG, "NULL bitmap_out");
  SelParams p;
  memset(&p, 0, sizeof(p));
  p.col = col->data;
  p.n = col->n;
  p.dtype = col->dtype;
  p.is_f64 = col->dtype == OCL_F64;
  p.anti = pred->anti ? 1 : 0;
  p.vec_ok = ((uintptr_t)col->data % 16) == 0;
  normalise_range(*pred, &p.lo, &p.hi, &p.flo, &p.fhi);
  p.out = bitmap_out;
  OCL_CUDA(launch_select_bitmap(p, ctx->grid, (cudaStream_t)stream), "select_bitmap launch");
  return OCL_OK;
}

ocl_status ocl_bitmap_combine(ocl_ctx* ctx, int32_t op, const uint32_t* a, const uint32_t* b, uint32_t* out, int64_t n,
                              void* stream) {
  if (!ctx) return fail(OCL_ERR_INVALID_ARG, "NULL ctx");
  if (op < 0 || op > 2) return fail(OCL_ERR_INVALID_ARG, "bad op %d", op);
  if (n < 0 || n >= kMaxRows) return fail(OCL_ERR_INVALID_ARG, "n out of range");
  if (n > 0 && (!a || !b || !out)) return fail(OCL_ERR_INVALID_ARG, "NULL bitmap");
  OCL_CUDA(launch_bitmap_combine(op, a, b, out, n, ctx->grid, (cudaStream_t)stream), "bitmap_combine launch");
  return OCL_OK;
}

// ---------------------------------------------------------------- a2
ocl_status ocl_prefix_compact_workspace_size(ocl_ctx* ctx, int64_t n, size_t* bytes) {
  if (!bytes) return fail(OCL_ERR_INVALID_ARG, "NULL bytes");
  if (n < 0 || n >= kMaxRows) return fail(OCL_ERR_INVALID_ARG, "n out of range");
  *bytes = prefix_compact_ws_bytes(n);
  return OCL_OK;
}

ocl_status ocl_prefix_compact(ocl_ctx* ctx, const uint32_t* bitmap, int64_t n, uint32_t* oids_out, int64_t* m_out,
                              void* ws, size_t ws_bytes, void* stream) {
  if (!ctx || !m_out) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/m_out");
  if (n < 0 || n >= kMaxRows) return fail(OCL_ERR_INVALID_ARG, "n out of range");
  if (n > 0 && (!bitmap || !oids_out || !ws)) return fail(OCL_ERR_INVALID_ARG, "NULL bitmap/oids_out/ws");
  if (n > 0 && ws_bytes < prefix_compact_ws_bytes(n)) return fail(OCL_ERR_CAPACITY, "workspace too small");
  int grid = ctx->sms * 4;
  OCL_CUDA(launch_prefix_compact(bitmap, n, oids_out, m_out, ws, grid, (cudaStream_t)stream), "prefix_compact launch");
  return OCL_OK;
}

// ---------------------------------------------------------------- a3
ocl_status ocl_gather(ocl_ctx* ctx, const ocl_column* col, const uint32_t* oids, const int64_t* m_dev, int64_t max_m,
                      void* out, void* stream) {
  if (!ctx) return fail(OCL_ERR_INVALID_ARG, "NULL ctx");
  ocl_status s = check_column(col, "col");
  if (s) return s;
  if (max_m < 0 || max_m >= kMaxRows) return fail(OCL_ERR_INVALID_ARG, "max_m out of range");
  if (max_m > 0 && (!oids || !out)) return fail(OCL_ERR_INVALID_ARG, "NULL oids/out");
  OCL_CUDA(launch_gather(col->data, dtype_width(col->dtype), oids, m_dev, max_m, out, ctx->grid, (cudaStream_t)stream),
           "gather launch");
  return OCL_OK;
}

// ---------------------------------------------------------------- a4-a6
static uint64_t group_cap(int64_t expected) { return next_pow2((uint64_t)std::max<int64_t>(2 * std::max<int64_t>(expected, 1), 16)); }

ocl_status ocl_group_build_workspace_size(ocl_ctx* ctx, int64_t max_rows, int64_t expected_groups, size_t* bytes) {
  if (!ctx || !bytes) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/bytes");
  if (expected_groups > ((int64_t)1 << 31)) return fail(OCL_ERR_UNSUPPORTED, "expected_groups > 2^31");
  *bytes = align_up((group_cap(expected_groups) + 1) * 16, 256) + align_up(emit_ws_bytes(ctx->grid), 256);
  return OCL_OK;
}

ocl_status ocl_group_build(ocl_ctx* ctx, const ocl_column* keys, int32_t nkeys, const uint32_t* oids,
                           const int64_t* m_dev, int64_t max_rows, int64_t expected_groups, int32_t* gid_out,
                           int64_t* keys_out, int64_t out_capacity, int64_t* ngroups_out, int32_t* dev_status,
                           void* ws, size_t ws_bytes, void* stream) {
  if (!ctx || !ngroups_out) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/ngroups_out");
  if (nkeys < 1) return fail(OCL_ERR_INVALID_ARG, "nkeys=%d (1..2)", nkeys);
  if (max_rows < 0 || max_rows >= kMaxRows) return fail(OCL_ERR_INVALID_ARG, "max_rows out of range");
  if (max_rows > 0 && !gid_out) return fail(OCL_ERR_INVALID_ARG, "NULL gid_out");
  Plan p;
  memset(&p, 0, sizeof(p));
  ocl_status s = plan_keys(keys, nkeys, p);
  if (s) return s;
  size_t need = 0;
  if ((s = ocl_group_build_workspace_size(ctx, max_rows, expected_groups, &need))) return s;
  if (!ws || ws_bytes < need) return fail(OCL_ERR_CAPACITY, "workspace %zu B < required %zu B", ws_bytes, need);
  uint64_t cap = group_cap(expected_groups);
  size_t tbytes = align_up((cap + 1) * 16, 256);
  cudaStream_t st = (cudaStream_t)stream;
  p.table = (uint8_t*)ws;
  p.mask = cap - 1;
  p.stride = 16;
  p.status = dev_status;
  p.oids = oids;
  p.m_dev = m_dev;
  p.n = max_rows;
  OCL_CUDA(cudaMemsetAsync(ws, 0, tbytes, st), "table init");
  if (dev_status) OCL_CUDA(cudaMemsetAsync(dev_status, 0, 4, st), "status init");
  OCL_CUDA(cudaMemsetAsync(ngroups_out, 0, 8, st), "group count init");
  OCL_CUDA(launch_group_build(p, gid_out, max_rows, ngroups_out, keys_out, keys_out ? out_capacity : INT64_MAX,
                              ctx->grid, st), "group build");
  return OCL_OK;
}

ocl_status ocl_group_build_paper_workspace_size(ocl_ctx* ctx, int64_t max_rows, int64_t expected_groups,
                                                size_t* bytes) {
  if (!ctx || !bytes) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/bytes");
  if (max_rows < 0 || max_rows >= kMaxRows) return fail(OCL_ERR_INVALID_ARG, "max_rows out of range");
  if (expected_groups > ((int64_t)1 << 31)) return fail(OCL_ERR_UNSUPPORTED, "expected_groups > 2^31");
  *bytes = hp_ws_bytes(max_rows, expected_groups);
  return OCL_OK;
}

ocl_status ocl_group_build_paper(ocl_ctx* ctx, const ocl_column* keys, int32_t nkeys, const uint32_t* oids,
                                 const int64_t* m_dev, int64_t max_rows, int64_t expected_groups, int32_t* gid_out,
                                 int64_t* keys_out, int64_t out_capacity, int64_t* ngroups_out, int32_t* dev_status,
                                 void* ws, size_t ws_bytes, void* stream) {
  if (!ctx || !ngroups_out) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/ngroups_out");
  if (nkeys < 1) return fail(OCL_ERR_INVALID_ARG, "nkeys=%d (1..2)", nkeys);
  size_t need = 0;
  ocl_status s = ocl_group_build_paper_workspace_size(ctx, max_rows, expected_groups, &need);
  if (s) return s;
  if (max_rows > 0 && !gid_out) return fail(OCL_ERR_INVALID_ARG, "NULL gid_out");
  Plan p;
  memset(&p, 0, sizeof(p));
  if ((s = plan_keys(keys, nkeys, p))) return s;
  if (!ws || ws_bytes < need) return fail(OCL_ERR_CAPACITY, "workspace %zu B < required %zu B", ws_bytes, need);
  cudaStream_t st = (cudaStream_t)stream;
  p.status = dev_status;
  p.oids = oids;
  p.m_dev = m_dev;
  p.n = max_rows;
  if (dev_status) OCL_CUDA(cudaMemsetAsync(dev_status, 0, 4, st), "status init");
  OCL_CUDA(launch_group_build_paper(p, expected_groups, gid_out, keys_out, keys_out ? out_capacity : INT64_MAX,
                                    ngroups_out, ws, ctx->sms, st), "paper group build");
  return OCL_OK;
}

ocl_status ocl_group_build_sorted_workspace_size(ocl_ctx* ctx, int64_t max_rows, size_t* bytes) {
  if (!ctx || !bytes) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/bytes");
  if (max_rows < 0 || max_rows > ((int64_t)1 << 31)) return fail(OCL_ERR_UNSUPPORTED, "max_rows outside [0, 2^31]");
  *bytes = group_build_sorted_ws_bytes(max_rows);
  return OCL_OK;
}

ocl_status ocl_group_build_sorted(ocl_ctx* ctx, const ocl_column* keys, int32_t nkeys, const uint32_t* oids,
                                  const int64_t* m_dev, int64_t max_rows, int32_t* gid_out, int64_t* keys_out,
                                  int64_t out_capacity, int64_t* ngroups_out, int32_t* dev_status, void* ws,
                                  size_t ws_bytes, void* stream) {
  if (!ctx || !ngroups_out) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/ngroups_out");
  if (nkeys < 1) return fail(OCL_ERR_INVALID_ARG, "nkeys=%d (1..2)", nkeys);
  if (out_capacity < 0) return fail(OCL_ERR_INVALID_ARG, "out_capacity < 0");
  size_t need = 0;
  ocl_status s = ocl_group_build_sorted_workspace_size(ctx, max_rows, &need);
  if (s) return s;
  if (max_rows > 0 && !gid_out) return fail(OCL_ERR_INVALID_ARG, "NULL gid_out");
  Plan p;
  memset(&p, 0, sizeof(p));
  if ((s = plan_keys(keys, nkeys, p))) return s;
  if (!oids)
    for (int i = 0; i < nkeys; ++i)
      if (keys[i].n < max_rows) return fail(OCL_ERR_INVALID_ARG, "key column shorter than max_rows");
  if (max_rows > 0 && (!ws || ws_bytes < need)) return fail(OCL_ERR_CAPACITY, "workspace %zu B < required %zu B", ws_bytes, need);
  cudaStream_t st = (cudaStream_t)stream;
  p.status = dev_status;
  p.oids = oids;
  p.m_dev = m_dev;
  p.n = max_rows;
  if (dev_status) OCL_CUDA(cudaMemsetAsync(dev_status, 0, 4, st), "status init");
  OCL_CUDA(launch_group_build_sorted(p, gid_out, keys_out, out_capacity, ngroups_out, ws, ctx->sms, st),
           "sorted group build");
  return OCL_OK;
}

// ---------------------------------------------------------------- equi hash join
static ocl_status join_key(const ocl_column* c, const char* what, DevKey* k) {
  ocl_status s = check_column(c, what);
  if (s) return s;
  if (c->dtype == OCL_F64) return fail(OCL_ERR_INVALID_ARG, "%s: f64 join key", what);
  const int w = 8 * dtype_width(c->dtype);
  k->col = devcol(*c);
  k->shift = 0;
  k->mask = w == 64 ? ~0ULL : ((1ULL << w) - 1);
  return OCL_OK;
}

ocl_status ocl_join_build_workspace_size(ocl_ctx* ctx, int64_t n_build, size_t* bytes) {
  if (!ctx || !bytes) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/bytes");
  if (n_build < 0 || n_build >= kMaxRows) return fail(OCL_ERR_INVALID_ARG, "n_build out of range");
  *bytes = join_build_ws_bytes(n_build);
  return OCL_OK;
}

ocl_status ocl_join_build(ocl_ctx* ctx, const ocl_column* build_key, void* build_ws, size_t build_ws_bytes,
                          int32_t* dev_status, void* stream) {
  if (!ctx) return fail(OCL_ERR_INVALID_ARG, "NULL ctx");
  DevKey k;
  ocl_status s = join_key(build_key, "build_key", &k);
  if (s) return s;
  if (!build_ws || build_ws_bytes < join_build_ws_bytes(build_key->n))
    return fail(OCL_ERR_CAPACITY, "build workspace %zu B < required %zu B", build_ws_bytes, join_build_ws_bytes(build_key->n));
  cudaStream_t st = (cudaStream_t)stream;
  if (dev_status) OCL_CUDA(cudaMemsetAsync(dev_status, 0, 4, st), "status init");
  OCL_CUDA(launch_join_build(k, build_key->n, build_ws, dev_status, ctx->sms, st), "join build");
  return OCL_OK;
}

ocl_status ocl_join_probe_workspace_size(ocl_ctx* ctx, int64_t max_rows, size_t* bytes) {
  if (!ctx || !bytes) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/bytes");
  if (max_rows < 0 || max_rows >= kMaxRows) return fail(OCL_ERR_INVALID_ARG, "max_rows out of range");
  *bytes = join_probe_ws_bytes(max_rows);
  return OCL_OK;
}

ocl_status ocl_join_probe(ocl_ctx* ctx, const ocl_column* build_key, const void* build_ws,
                          const ocl_column* probe_key, const uint32_t* probe_oids, const int64_t* m_dev,
                          int64_t max_rows, int32_t pk_build, uint32_t* out_probe, uint32_t* out_build,
                          int64_t out_capacity, int64_t* nout_dev, int32_t* dev_status, void* ws, size_t ws_bytes,
                          void* stream) {
  if (!ctx || !nout_dev) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/nout_dev");
  DevKey bk, pk;
  ocl_status s = join_key(build_key, "build_key", &bk);
  if (s) return s;
  if ((s = join_key(probe_key, "probe_key", &pk))) return s;
  if (build_key->dtype != probe_key->dtype) return fail(OCL_ERR_INVALID_ARG, "build/probe key dtypes differ");
  if (max_rows < 0 || max_rows >= kMaxRows) return fail(OCL_ERR_INVALID_ARG, "max_rows out of range");
  if (!probe_oids && probe_key->n < max_rows) return fail(OCL_ERR_INVALID_ARG, "probe column shorter than max_rows");
  if (out_capacity < 0 || (out_capacity > 0 && (!out_probe || !out_build))) return fail(OCL_ERR_INVALID_ARG, "bad outputs");
  if (!build_ws) return fail(OCL_ERR_INVALID_ARG, "NULL build_ws");
  if (max_rows > 0 && (!ws || ws_bytes < join_probe_ws_bytes(max_rows)))
    return fail(OCL_ERR_CAPACITY, "workspace %zu B < required %zu B", ws_bytes, join_probe_ws_bytes(max_rows));
  cudaStream_t st = (cudaStream_t)stream;
  if (dev_status) OCL_CUDA(cudaMemsetAsync(dev_status, 0, 4, st), "status init");
  OCL_CUDA(launch_join_probe(build_ws, build_key->n, pk, probe_oids, m_dev, max_rows, pk_build != 0, out_probe,
                             out_build, out_capacity, nout_dev, dev_status, ws, ctx->sms, st), "join probe");
  return OCL_OK;
}

// ---------------------------------------------------------------- a7-a8
ocl_status ocl_group_aggregate_workspace_size(ocl_ctx* ctx, int64_t max_groups, const ocl_column* vals, int32_t nvals,
                                              const ocl_agg* aggs, int32_t naggs, size_t* bytes) {
  if (!ctx || !bytes) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/bytes");
  if (max_groups < 0 || max_groups >= kMaxRows) return fail(OCL_ERR_INVALID_ARG, "max_groups out of range");
  Planned P;
  memset(&P, 0, sizeof(P));
  ocl_status s = plan_values(vals, nvals, aggs, naggs, &P);
  if (s) return s;
  *bytes = align_up((size_t)max_groups * P.plan.stride, 256) + 256;
  return OCL_OK;
}

ocl_status ocl_group_aggregate(ocl_ctx* ctx, const int32_t* gids, const uint32_t* oids, const int64_t* m_dev,
                               int64_t max_rows, const int64_t* ngroups_dev, int64_t max_groups,
                               const ocl_column* vals, int32_t nvals, const ocl_agg* aggs, int32_t naggs, void* ws,
                               size_t ws_bytes, void* stream) {
  if (!ctx) return fail(OCL_ERR_INVALID_ARG, "NULL ctx");
  if (max_rows < 0 || max_rows >= kMaxRows) return fail(OCL_ERR_INVALID_ARG, "max_rows out of range");
  if (max_rows > 0 && !gids) return fail(OCL_ERR_INVALID_ARG, "NULL gids");
  Planned P;
  memset(&P, 0, sizeof(P));
  ocl_status s = plan_values(vals, nvals, aggs, naggs, &P);
  if (s) return s;
  size_t need = 0;
  if ((s = ocl_group_aggregate_workspace_size(ctx, max_groups, vals, nvals, aggs, naggs, &need))) return s;
  if (max_groups > 0 && (!ws || ws_bytes < need)) return fail(OCL_ERR_CAPACITY, "workspace %zu B < required %zu B", ws_bytes, need);
  if (!oids) {
    for (int i = 0; i < nvals; ++i)
      if (vals[i].n < max_rows) return fail(OCL_ERR_INVALID_ARG, "value column shorter than max_rows");
  }
  cudaStream_t st = (cudaStream_t)stream;
  Plan& p = P.plan;
  p.table = (uint8_t*)ws;
  p.gids = gids;
  p.oids = oids;
  p.m_dev = m_dev;
  p.n = max_rows;
  if (max_groups == 0) return OCL_OK;
  OCL_CUDA(cudaMemsetAsync(ws, 0, (size_t)max_groups * p.stride, st), "state init");
  p.direct = 1;
  OCL_CUDA(launch_group_aggregate(p, max_rows, ngroups_dev, max_groups, P.values_f64, ctx->sms, st),
           "group_aggregate launch");
  P.fin.out_capacity = max_groups;
  OCL_CUDA(launch_finalize_dense(p.table, p.stride, ngroups_dev, max_groups, P.fin, ctx->grid, st), "finalize");
  return OCL_OK;
}

// ---------------------------------------------------------------- a9 fused
ocl_status ocl_select_group_aggregate_workspace_size(ocl_ctx* ctx, const ocl_sga_args* args, size_t* bytes) {
  if (!ctx || !bytes) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/bytes");
  Planned P;
  ocl_status s = plan_sga(args, &P, false);
  if (s) return s;
  if (args->distributed) return dist_ws_bytes(ctx, args, P, bytes);
  *bytes = sga_ws_bytes(ctx, P);
  return OCL_OK;
}

ocl_status ocl_select_group_aggregate(ocl_ctx* ctx, const ocl_sga_args* args, void* ws, size_t ws_bytes, void* stream) {
  if (!ctx) return fail(OCL_ERR_INVALID_ARG, "NULL ctx");
  Planned P;
  ocl_status s = plan_sga(args, &P);
  if (s) return s;
  cudaStream_t st = (cudaStream_t)stream;
  if (args->distributed) return run_distributed(ctx, args, P, ws, ws_bytes, st);
  NvtxRange nv("ocl:select+group+aggregate");
  if (P.sorted || P.sortgrp) return run_sortpath(ctx, args, P, ws, ws_bytes, st, nullptr, args->out_capacity,
                                                 args->ngroups_out);
  void* ews = nullptr;
  EmitArgs ea;
  memset(&ea, 0, sizeof(ea));
  ea.kind = EMIT_FINAL;
  ea.fin = P.fin;
  bool emitted = false;
  if ((s = run_fused(ctx, args, P, ws, ws_bytes, st, &ews, args->order_by_key ? nullptr : &ea, args->ngroups_out,
                     args->out_capacity, &emitted)))
    return s;
  if (!emitted)
    OCL_CUDA(launch_emit(P.plan.table, P.cap, P.plan.stride, ea, args->ngroups_out, args->out_capacity,
                         args->dev_status, args->order_by_key != 0, ews, ctx->grid, st), "finalize");
  return OCL_OK;
}

ocl_status ocl_select_group_aggregate_sync_workspace_size(ocl_ctx* ctx, const ocl_sga_args* args, size_t* bytes) {
  if (!ctx || !bytes || !args) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/args/bytes");
  int64_t egs[40];
  const int n = sync_ladder(args, egs, 40);
  ocl_sga_args a = *args;
  size_t best = 0;
  for (int i = 0; i < n; ++i) {
    a.expected_groups = egs[i];
    size_t b = 0;
    ocl_status s = ocl_select_group_aggregate_workspace_size(ctx, &a, &b);
    if (s) return s;
    best = std::max(best, b);
  }
  *bytes = align_up(best, 256) + (args->dev_status ? 0 : 256);
  return OCL_OK;
}

ocl_status ocl_select_group_aggregate_sync(ocl_ctx* ctx, const ocl_sga_args* args, void* ws, size_t ws_bytes,
                                           void* stream) {
  size_t need = 0;
  ocl_status s = ocl_select_group_aggregate_sync_workspace_size(ctx, args, &need);
  if (s) return s;
  if (!ws || ws_bytes < need) return fail(OCL_ERR_CAPACITY, "workspace %zu B < required %zu B", ws_bytes, need);
  cudaStream_t st = (cudaStream_t)stream;
  ocl_sga_args a = *args;
  if (!a.dev_status) a.dev_status = (int32_t*)((uint8_t*)ws + need - 256);
  int64_t egs[40];
  const int n = sync_ladder(args, egs, 40);
  for (int i = 0; i < n;) {
    a.expected_groups = egs[i];
    if ((s = ocl_select_group_aggregate(ctx, &a, ws, ws_bytes, stream))) return s;
    int32_t hs = 0;
    int64_t G = 0;
    OCL_CUDA(cudaMemcpyAsync(&hs, a.dev_status, 4, cudaMemcpyDeviceToHost, st), "status readback");
    OCL_CUDA(cudaMemcpyAsync(&G, a.ngroups_out, 8, cudaMemcpyDeviceToHost, st), "group count readback");
    OCL_CUDA(cudaStreamSynchronize(st), "sync");
    if (hs == OCL_OK) return OCL_OK;
    if (hs != OCL_ERR_CAPACITY) return fail((ocl_status)hs, "device status %d", hs);
    if (G > a.out_capacity)
      return fail(OCL_ERR_CAPACITY, "%lld groups > out_capacity %lld", (long long)G, (long long)a.out_capacity);
    // the table overflowed: restart at the ladder step covering max(4 x, 2 G)
    const int64_t want = std::max<int64_t>(4 * egs[i], 2 * G);
    int j = i + 1;
    while (j < n - 1 && egs[j] < want) ++j;
    if (j >= n) return fail(OCL_ERR_CAPACITY, "hash table full at expected_groups=%lld (out_capacity %lld)",
                            (long long)egs[i], (long long)a.out_capacity);
    i = j;
  }
  return fail(OCL_ERR_CAPACITY, "hash table full");
}

// ---------------------------------------------------------------- a10 multi-GPU pieces
ocl_status ocl_partial_row_bytes(const ocl_sga_args* args, size_t* bytes) {
  if (!bytes) return fail(OCL_ERR_INVALID_ARG, "NULL bytes");
  Planned P;
  ocl_status s = plan_sga(args, &P, false);
  if (s) return s;
  *bytes = (size_t)P.plan.stride;
  return OCL_OK;
}

ocl_status ocl_sga_partial(ocl_ctx* ctx, const ocl_sga_args* args, void* partial_out, int64_t partial_capacity,
                           int64_t* npartial_out, void* ws, size_t ws_bytes, void* stream) {
  if (!ctx || !npartial_out) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/npartial_out");
  if (partial_capacity < 0 || (partial_capacity > 0 && !partial_out)) return fail(OCL_ERR_INVALID_ARG, "bad partial_out");
  Planned P;
  ocl_status s = plan_sga(args, &P, false);
  if (s) return s;
  if (args->distributed) return fail(OCL_ERR_INVALID_ARG, "ocl_sga_partial is the local step: distributed must be 0");
  NvtxRange nv("ocl:partial");
  return local_partial(ctx, args, P, ws, ws_bytes, (cudaStream_t)stream, (uint8_t*)partial_out, partial_capacity,
                       npartial_out);
}

static uint64_t merge_cap(const ocl_sga_args* args, int32_t nparts, int64_t part_capacity) {
  int64_t bound = (int64_t)nparts * part_capacity;
  return next_pow2((uint64_t)std::max<int64_t>(2 * std::max<int64_t>(bound, 1), 16));
}

ocl_status ocl_merge_partials_workspace_size(ocl_ctx* ctx, const ocl_sga_args* args, int32_t nparts,
                                             int64_t part_capacity, size_t* bytes) {
  if (!ctx || !bytes) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/bytes");
  if (nparts < 0 || part_capacity < 0) return fail(OCL_ERR_INVALID_ARG, "bad nparts/part_capacity");
  Planned P;
  ocl_status s = plan_sga(args, &P, false);
  if (s) return s;
  uint64_t cap = merge_cap(args, nparts, part_capacity);
  *bytes = align_up((cap + 1) * (size_t)P.plan.stride, 256) + align_up(emit_ws_bytes(ctx->grid), 256);
  return OCL_OK;
}

ocl_status ocl_merge_partials(ocl_ctx* ctx, const ocl_sga_args* args, const void* partials, int32_t nparts,
                              int64_t part_capacity, const int64_t* part_counts, void* ws, size_t ws_bytes,
                              void* stream) {
  if (!ctx) return fail(OCL_ERR_INVALID_ARG, "NULL ctx");
  if (nparts < 0 || part_capacity < 0) return fail(OCL_ERR_INVALID_ARG, "bad nparts/part_capacity");
  if (nparts > 0 && part_capacity > 0 && (!partials || !part_counts)) return fail(OCL_ERR_INVALID_ARG, "NULL partials");
  Planned P;
  ocl_status s = plan_sga(args, &P);
  if (s) return s;
  size_t need = 0;
  if ((s = ocl_merge_partials_workspace_size(ctx, args, nparts, part_capacity, &need))) return s;
  if (!ws || ws_bytes < need) return fail(OCL_ERR_CAPACITY, "workspace %zu B < required %zu B", ws_bytes, need);
  uint64_t cap = merge_cap(args, nparts, part_capacity);
  if (args->order_by_key && !sorted_emit_supported(cap))
    return fail(OCL_ERR_UNSUPPORTED, "order_by_key with %llu merge slots", (unsigned long long)cap);
  size_t tbytes = align_up((cap + 1) * (size_t)P.plan.stride, 256);
  cudaStream_t st = (cudaStream_t)stream;
  OCL_CUDA(cudaMemsetAsync(ws, 0, tbytes, st), "merge table init");
  if (args->dev_status) OCL_CUDA(cudaMemsetAsync(args->dev_status, 0, 4, st), "status init");
  OCL_CUDA(launch_merge_partials((const uint8_t*)partials, nparts, part_capacity, part_counts, P.fin, (uint8_t*)ws,
                                 cap - 1, args->dev_status, ctx->grid, st), "merge");
  EmitArgs ea;
  memset(&ea, 0, sizeof(ea));
  ea.kind = EMIT_FINAL;
  ea.fin = P.fin;
  OCL_CUDA(launch_emit((uint8_t*)ws, cap, P.plan.stride, ea, args->ngroups_out, args->out_capacity, args->dev_status,
                       args->order_by_key != 0, (uint8_t*)ws + tbytes, ctx->grid, st), "merge finalize");
  return OCL_OK;
}

ocl_status ocl_radix_sort_workspace_size(ocl_ctx* ctx, int64_t n, int32_t with_payload, int32_t with_rowids,
                                         size_t* bytes) {
  if (!ctx || !bytes) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/bytes");
  if (n < 0 || n >= kMaxRows) return fail(OCL_ERR_INVALID_ARG, "n out of range");
  *bytes = radix_ws_bytes(n, with_payload != 0, with_rowids != 0);
  return OCL_OK;
}

ocl_status ocl_radix_sort(ocl_ctx* ctx, const ocl_column* keys, int32_t nkeys, const ocl_column* payload,
                          uint64_t* keys_out, void* payload_out, uint32_t* rowids_out, void* ws, size_t ws_bytes,
                          void* stream) {
  if (!ctx) return fail(OCL_ERR_INVALID_ARG, "NULL ctx");
  if (nkeys < 1) return fail(OCL_ERR_INVALID_ARG, "nkeys=%d (1..2)", nkeys);
  Plan p;
  memset(&p, 0, sizeof(p));
  ocl_status s = plan_keys(keys, nkeys, p);
  if (s) return s;
  const int64_t n = keys[0].n;
  for (int i = 1; i < nkeys; ++i)
    if (keys[i].n != n) return fail(OCL_ERR_INVALID_ARG, "key columns differ in length");
  if (payload) {
    if ((s = check_column(payload, "payload"))) return s;
    if (dtype_width(payload->dtype) != 8 || payload->n != n) return fail(OCL_ERR_INVALID_ARG, "payload: 8-byte column of n rows");
    if (n > 0 && !payload_out) return fail(OCL_ERR_INVALID_ARG, "NULL payload_out");
  }
  if (n > 0 && !keys_out) return fail(OCL_ERR_INVALID_ARG, "NULL keys_out");
  const size_t need = radix_ws_bytes(n, payload != nullptr, rowids_out != nullptr);
  if (n > 0 && (!ws || ws_bytes < need)) return fail(OCL_ERR_CAPACITY, "workspace %zu B < required %zu B", ws_bytes, need);
  p.n = n;
  OCL_CUDA(launch_radix(p, payload ? (const uint64_t*)payload->data : nullptr, keys_out,
                        payload ? (uint64_t*)payload_out : nullptr, rowids_out, ws, ctx->sms, (cudaStream_t)stream),
           "radix sort");
  return OCL_OK;
}

ocl_status ocl_route_partials_workspace_size(ocl_ctx* ctx, int32_t nparts, size_t* bytes) {
  if (!ctx || !bytes) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/bytes");
  if (nparts < 1 || nparts > route_max_parts()) return fail(OCL_ERR_INVALID_ARG, "nparts=%d (1..%d)", nparts, route_max_parts());
  *bytes = route_ws_bytes(nparts);
  return OCL_OK;
}

ocl_status ocl_route_partials(ocl_ctx* ctx, const void* rows, const int64_t* nrows_dev, int64_t max_rows,
                              int32_t row_bytes, int32_t nparts, void* out, int64_t* part_counts, void* ws,
                              size_t ws_bytes, void* stream) {
  size_t need = 0;
  ocl_status s = ocl_route_partials_workspace_size(ctx, nparts, &need);
  if (s) return s;
  if (max_rows < 0) return fail(OCL_ERR_INVALID_ARG, "max_rows < 0");
  if (row_bytes < 16 || row_bytes % 8) return fail(OCL_ERR_INVALID_ARG, "row_bytes=%d (multiple of 8, >= 16)", row_bytes);
  if (!part_counts || !ws) return fail(OCL_ERR_INVALID_ARG, "NULL part_counts/ws");
  if (max_rows > 0 && (!rows || !out)) return fail(OCL_ERR_INVALID_ARG, "NULL rows/out");
  if (ws_bytes < need) return fail(OCL_ERR_CAPACITY, "workspace %zu B < required %zu B", ws_bytes, need);
  OCL_CUDA(launch_route(rows, nrows_dev, max_rows, row_bytes, nparts, out, part_counts, ws, ctx->sms,
                        (cudaStream_t)stream), "route partials");
  return OCL_OK;
}

// ---------------------------------------------------------------- end to end from host buffers
namespace {
struct HostCols {
  int ncols;
  const void* host[3 * kMaxVals + kMaxPreds + kMaxKeys];
  int width[3 * kMaxVals + kMaxPreds + kMaxKeys];
  size_t off[3 * kMaxVals + kMaxPreds + kMaxKeys];   // offset inside one staging slot
  size_t slot_bytes;
};

int host_col_index(HostCols& h, const void* ptr, int width, int64_t chunk_rows) {
  for (int i = 0; i < h.ncols; ++i)
    if (h.host[i] == ptr) return i;
  int i = h.ncols++;
  h.host[i] = ptr;
  h.width[i] = width;
  h.off[i] = h.slot_bytes;
  h.slot_bytes += align_up((size_t)chunk_rows * width, 256);
  return i;
}

void collect_host_cols(const Planned& P, HostCols& h, int64_t chunk_rows) {
  memset(&h, 0, sizeof(h));
  const Plan& p = P.plan;
  for (int i = 0; i < p.npreds; ++i) host_col_index(h, p.preds[i].col.ptr, p.preds[i].col.width, chunk_rows);
  for (int i = 0; i < p.nkeys; ++i) host_col_index(h, p.keys[i].col.ptr, p.keys[i].col.width, chunk_rows);
  for (int v = 0; v < p.nvals; ++v) {
    host_col_index(h, p.vals[v].a.ptr, p.vals[v].a.width, chunk_rows);
    if (p.vals[v].expr >= OCL_EXPR_MUL_1MINUS) host_col_index(h, p.vals[v].b.ptr, p.vals[v].b.width, chunk_rows);
    if (p.vals[v].expr >= OCL_EXPR_MUL_1MINUS_1PLUS) host_col_index(h, p.vals[v].c.ptr, p.vals[v].c.width, chunk_rows);
  }
}

size_t host_out_bytes(const ocl_sga_args* a, const Planned& P) {
  size_t b = align_up((size_t)a->out_capacity * 8, 256) + 256;   // keys + (ngroups, status)
  for (int i = 0; i < a->naggs; ++i) {
    size_t es = (a->aggs[i].op == OCL_AGG_SUM && !P.fin.aggs[i].is_f64) ? 16 : 8;
    b += align_up((size_t)a->out_capacity * es, 256);
  }
  return b;
}
}  // namespace

ocl_status ocl_select_group_aggregate_host_workspace_size(ocl_ctx* ctx, const ocl_sga_args* args, int64_t chunk_rows,
                                                          size_t* bytes) {
  if (!ctx || !bytes) return fail(OCL_ERR_INVALID_ARG, "NULL ctx/bytes");
  if (chunk_rows <= 0 || (chunk_rows & 1023)) return fail(OCL_ERR_INVALID_ARG, "chunk_rows must be a positive multiple of 1024");
  Planned P;
  ocl_status s = plan_sga(args, &P, false);
  if (s) return s;
  if (P.sorted || P.sortgrp) return fail(OCL_ERR_UNSUPPORTED, "sort-based grouping is not available on the host-buffer path");
  P.pbits = -1;             // chunks stream through the one-pass fused kernel
  HostCols h;
  collect_host_cols(P, h, chunk_rows);
  *bytes = sga_ws_bytes(ctx, P) + 2 * h.slot_bytes + host_out_bytes(args, P);
  if (args->distributed) {         // + the exchange region after the host-path workspace
    DistLayout L;
    if ((s = dist_layout(ctx, args, P, *bytes, &L))) return s;
    *bytes = L.total;
  }
  return OCL_OK;
}

ocl_status ocl_select_group_aggregate_host(ocl_ctx* ctx, const ocl_sga_args* args, int64_t chunk_rows, void* ws,
                                           size_t ws_bytes, void* stream) {
  if (!ctx) return fail(OCL_ERR_INVALID_ARG, "NULL ctx");
  if (args && args->bitmap_out) return fail(OCL_ERR_INVALID_ARG, "bitmap_out must be NULL on the host path");
  size_t need = 0;
  ocl_status s = ocl_select_group_aggregate_host_workspace_size(ctx, args, chunk_rows, &need);
  if (s) return s;
  if (!ws || ws_bytes < need) return fail(OCL_ERR_CAPACITY, "workspace %zu B < required %zu B", ws_bytes, need);
  Planned P;
  if ((s = plan_sga(args, &P))) return s;
  P.pbits = -1;
  HostCols h;
  collect_host_cols(P, h, chunk_rows);
  // carve: [table | emit ws] [staging slot 0] [staging slot 1] [device outputs]
  uint8_t* base = (uint8_t*)ws;
  uint8_t* table = base;
  uint8_t* ews = base + P.table_bytes;
  uint8_t* slot[2] = {base + sga_ws_bytes(ctx, P), base + sga_ws_bytes(ctx, P) + h.slot_bytes};
  uint8_t* outs = slot[1] + h.slot_bytes;
  int64_t* d_ngroups = (int64_t*)outs;
  int32_t* d_status = (int32_t*)(outs + 8);
  int64_t* d_keys = (int64_t*)(outs + 256);
  uint8_t* cur = outs + 256 + align_up((size_t)args->out_capacity * 8, 256);
  FinPlan fin = P.fin;
  fin.keys_out = args->keys_out ? d_keys : nullptr;
  fin.ngroups_out = d_ngroups;
  fin.status = d_status;
  size_t out_es[kMaxAggs];
  for (int i = 0; i < args->naggs; ++i) {
    out_es[i] = (args->aggs[i].op == OCL_AGG_SUM && !P.fin.aggs[i].is_f64) ? 16 : 8;
    fin.aggs[i].out = cur;
    cur += align_up((size_t)args->out_capacity * out_es[i], 256);
  }
  cudaStream_t user = (cudaStream_t)stream;
  cudaStream_t cs = ctx->copy_stream, ks = ctx->comp_stream;
  OCL_CUDA(cudaStreamSynchronize(user), "sync caller stream");
  OCL_CUDA(cudaMemsetAsync(table, 0, P.table_bytes, ks), "table init");
  OCL_CUDA(cudaMemsetAsync(d_status, 0, 4, ks), "status init");
  OCL_CUDA(cudaEventRecord(ctx->ev_consumed[0], ks), "event");
  OCL_CUDA(cudaEventRecord(ctx->ev_consumed[1], ks), "event");
  // distributed: the exchange region follows the host-path workspace; the chunks' table
  // overflow goes to the header's status word so that every rank sees it
  DistLayout L;
  memset(&L, 0, sizeof(L));
  int64_t* hdr = nullptr;
  if (args->distributed) {
    if ((s = dist_layout(ctx, args, P, (size_t)(cur - base), &L))) return s;
    hdr = (int64_t*)(base + L.off_hdr);
    OCL_CUDA(cudaMemsetAsync(hdr, 0, (size_t)L.W * 8, ks), "header init");
  }
  Plan p = P.plan;
  p.table = table;
  p.status = hdr ? (int32_t*)&hdr[L.W - 1] : d_status;
  p.bitmap_out = nullptr;
  const int mode = fused_mode(args);
  const int64_t n = P.plan.n;
  int64_t nchunks = (n + chunk_rows - 1) / chunk_rows;
  for (int64_t c = 0; c < nchunks; ++c) {
    int sl = (int)(c & 1);
    int64_t r0 = c * chunk_rows, rows = std::min<int64_t>(chunk_rows, n - r0);
    OCL_CUDA(cudaStreamWaitEvent(cs, ctx->ev_consumed[sl], 0), "wait");
    for (int i = 0; i < h.ncols; ++i)
      OCL_CUDA(cudaMemcpyAsync(slot[sl] + h.off[i], (const uint8_t*)h.host[i] + r0 * h.width[i],
                               (size_t)rows * h.width[i], cudaMemcpyHostToDevice, cs), "H2D chunk");
    OCL_CUDA(cudaEventRecord(ctx->ev_copied[sl], cs), "event");
    OCL_CUDA(cudaStreamWaitEvent(ks, ctx->ev_copied[sl], 0), "wait");
    // re-point the plan's columns into this staging slot
    Plan q = p;
    q.n = rows;
    auto remap = [&](DevCol& dc) {
      for (int i = 0; i < h.ncols; ++i)
        if (h.host[i] == dc.ptr) { dc.ptr = slot[sl] + h.off[i]; return; }
    };
    for (int i = 0; i < q.npreds; ++i) remap(q.preds[i].col);
    for (int i = 0; i < q.nkeys; ++i) remap(q.keys[i].col);
    for (int i = 0; i < q.ncols; ++i) remap(q.vcols[i]);
    for (int v = 0; v < q.nvals; ++v) {
      remap(q.vals[v].a);
      if (q.vals[v].expr >= OCL_EXPR_MUL_1MINUS) remap(q.vals[v].b);
      if (q.vals[v].expr >= OCL_EXPR_MUL_1MINUS_1PLUS) remap(q.vals[v].c);
    }
    q.vec_ok = 1;   // staging buffers are 256-byte aligned
    int kind = 0;
    OCL_CUDA(launch_fused(q, mode, P.values_f64, ctx->sms, ks, &kind), "fused kernel (chunk)");
    OCL_CUDA(cudaEventRecord(ctx->ev_consumed[sl], ks), "event");
  }
  if (args->distributed) {
    EmitArgs pa;
    memset(&pa, 0, sizeof(pa));
    pa.kind = EMIT_PARTIAL;
    pa.out_capacity = L.part_cap;
    pa.partial_out = base + L.off_part;
    pa.status = p.status;
    int64_t* pcount = L.mode == 1 ? hdr : (int64_t*)(base + L.off_pcount);
    OCL_CUDA(launch_emit(table, P.cap, p.stride, pa, pcount, L.part_cap, p.status, false, ews, ctx->grid, ks),
             "partial export");
    if ((s = dist_exchange_merge(ctx, args, L, base, fin, d_ngroups, d_status, ks))) return s;
  } else {
    EmitArgs ea;
    memset(&ea, 0, sizeof(ea));
    ea.kind = EMIT_FINAL;
    ea.fin = fin;
    OCL_CUDA(launch_emit(table, P.cap, p.stride, ea, d_ngroups, args->out_capacity, d_status,
                         args->order_by_key != 0, ews, ctx->grid, ks), "finalize");
  }
  // results back to the host
  OCL_CUDA(cudaMemcpyAsync(args->ngroups_out, d_ngroups, 8, cudaMemcpyDeviceToHost, ks), "D2H ngroups");
  if (args->dev_status) OCL_CUDA(cudaMemcpyAsync(args->dev_status, d_status, 4, cudaMemcpyDeviceToHost, ks), "D2H status");
  OCL_CUDA(cudaStreamSynchronize(ks), "sync");
  int64_t G = std::min<int64_t>(*args->ngroups_out, args->out_capacity);
  if (G > 0) {
    if (args->keys_out) OCL_CUDA(cudaMemcpyAsync(args->keys_out, d_keys, (size_t)G * 8, cudaMemcpyDeviceToHost, ks), "D2H keys");
    for (int i = 0; i < args->naggs; ++i)
      OCL_CUDA(cudaMemcpyAsync(args->aggs[i].out, fin.aggs[i].out, (size_t)G * out_es[i], cudaMemcpyDeviceToHost, ks), "D2H agg");
  }
  OCL_CUDA(cudaStreamSynchronize(ks), "sync");
  return OCL_OK;
}

}  // extern "C"
