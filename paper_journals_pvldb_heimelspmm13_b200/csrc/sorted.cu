// sorted.cu — GROUP BY on sorted input.
//
// Paper (§4.1.6): "If the input is sorted, we identify group
// boundaries by having each thread compare its value with its successor. Then, a
// prefix sum operation is used to generate dense group IDs."  No hash table: a
// group is a run of equal keys, its dense id is the number of runs before it, and
// ids come out in key order (so ORDER BY key is free).  "Sorted" = the packed key
// (unsigned 64-bit) is non-decreasing over all rows — MonetDB's
// tsorted property of the column; a decreasing step is detected on the device and
// reported as OCL_ERR_INVALID_ARG through the status word.
//
// Two operators:
//  * k_group_build_sorted (unfused a4, ocl_group_build_sorted): rows j < m with key
//    at oids[j]; head(j) = key(j) != key(j-1) (the paper's successor compare, seen
//    from the successor), one decoupled look-back prefix sum over the heads gives
//    gid(j) = #heads <= j - 1; keys_out[gid] written by the head rows.
//  * the fused select -> sorted group -> aggregate (ocl_sga_args.key_sorted), over
//    2048-row units, one warp per unit, 8 units per CTA tile:
//      pass 1 k_sorted_summary: the predicate and key columns of the unit -> its
//        summary (runs starting in it, first and last qualifying key); a row starts a
//        run when it qualifies and its key differs from the previous qualifying row's
//        key (selection does not break a run).  Summaries combine with the monoid
//        (runs_A + runs_B - [last_A == first_B], first, last); each CTA also writes
//        its tile's combined summary.
//      k_sorted_tiles (one CTA): exclusive prefix over the tile summaries; writes G.
//      pass 2 k_sorted_agg: a warp first derives its unit's prefix (tile prefix +
//        the summaries of the earlier units of its tile) -> the group id of the unit's
//        first run; then reads the unit again, all columns, in steps of 32*K rows (K
//        consecutive rows per lane).  A lane folds its rows; a warp segmented scan
//        over the lanes' open pieces (segments start at lanes holding a run start)
//        completes runs that cross lanes; runs closed in the step are staged in shared
//        memory and written by the warp as one range of output rows (gid = unit base +
//        run index).  No table, no atomics — except for the unit's first and last
//        run, which may continue into neighbouring units: those are merged (atomics)
//        into a small "chain" table keyed by gid.
//      k_sorted_chain_emit: finalises the chain table entries.
//    Algorithmic bytes: the columns once (pass 2) + predicate and key columns
//    (pass 1) + G output rows.
#include <stdlib.h>
#include <string.h>

#include <algorithm>

#include "sga_device.cuh"

namespace ocl {

constexpr int kSortedWarps = 8;
constexpr int kSortedThreads = kSortedWarps * 32;
constexpr int kSortedUnitRows = 2048;                 // rows per warp unit
constexpr int kSortedTileRows = kSortedWarps * kSortedUnitRows;
constexpr int kTileScanThreads = 1024;

// Run monoid of a row range: runs starting in it (its first qualifying row counts),
// first / last qualifying packed key, any row qualifies.
struct Mono {
  uint64_t runs, first, last, has;
};
__device__ __forceinline__ Mono mono_id() { return Mono{0, 0, 0, 0}; }
__device__ __forceinline__ Mono mono_combine(const Mono& a, const Mono& b) {
  Mono r;
  r.runs = a.runs + b.runs - ((a.has && b.has && a.last == b.first) ? 1 : 0);
  r.first = a.has ? a.first : b.first;
  r.last = b.has ? b.last : a.last;
  r.has = a.has | b.has;
  return r;
}
__device__ __forceinline__ Mono mono_shfl_down(const Mono& m, int d) {
  return Mono{__shfl_down_sync(0xffffffffu, m.runs, d), __shfl_down_sync(0xffffffffu, m.first, d),
              __shfl_down_sync(0xffffffffu, m.last, d), __shfl_down_sync(0xffffffffu, m.has, d)};
}
__device__ __forceinline__ Mono mono_shfl_up(const Mono& m, int d) {
  return Mono{__shfl_up_sync(0xffffffffu, m.runs, d), __shfl_up_sync(0xffffffffu, m.first, d),
              __shfl_up_sync(0xffffffffu, m.last, d), __shfl_up_sync(0xffffffffu, m.has, d)};
}
__device__ __forceinline__ Mono mono_bcast(const Mono& m, int src) {
  return Mono{__shfl_sync(0xffffffffu, m.runs, src), __shfl_sync(0xffffffffu, m.first, src),
              __shfl_sync(0xffffffffu, m.last, src), __shfl_sync(0xffffffffu, m.has, src)};
}
// Combination of the 32 lanes' values in lane order (lane 0 first), broadcast.
__device__ __forceinline__ Mono mono_warp_reduce(Mono m, int lane) {
#pragma unroll
  for (int d = 1; d < 32; d <<= 1) {
    const Mono y = mono_shfl_down(m, d);
    if (lane + d < 32) m = mono_combine(m, y);
  }
  return mono_bcast(m, 0);
}

// Integer COL outputs of the fast path, by kind (host-built from the FinPlan; ok = 0
// when the aggregate list does not fit this map, e.g. the same output twice).
struct FastEmit {
  int32_t ok, pad;
  int64_t* cnt;
  uint64_t* sum[kMaxVals];   // int128 {lo, hi}
  double* avg[kMaxVals];
  int64_t* mn[kMaxVals];
  int64_t* mx[kMaxVals];
};

struct SortedArgs {
  Mono* sum;                // per unit summary (pass 1)
  Mono* tile;               // per tile summary (pass 1), then the tile's exclusive prefix (k_sorted_tiles)
  uint8_t* chains;          // chain table: Plan::stride-byte entries keyed by gid (linear probing)
  uint64_t* chain_key;      // packed group key per chain-table slot
  uint64_t chain_mask;      // capacity - 1
  int64_t nunits, ntiles;
  int64_t* ngroups_out;
  int64_t out_capacity;
  int32_t* status;
  FinPlan fin;
  FastEmit fe;
  uint8_t* partial_out;     // non-null: write partial rows (multi-GPU export) instead of final outputs
};

__device__ __forceinline__ uint32_t lane_lt() {
  uint32_t m;
  asm("mov.u32 %0, %%lanemask_lt;" : "=r"(m));
  return m;
}

// ------------------------------------------------------------------ predicate + key of rows
template <class Sh>
__device__ __forceinline__ void qk_pair(const Plan& p, int64_t r, bool& q0, bool& q1, typename Sh::Key& k0,
                                        typename Sh::Key& k1) {
  q0 = q1 = true;
#pragma unroll
  for (int i = 0; i < kMaxPreds; ++i) {
    if (i >= Sh::np(p)) break;
    uint64_t u0, u1;
    ld2w(Sh::pw(p, i), p.preds[i].col.ptr, r, u0, u1);
    q0 = q0 && pred_ok<Sh>(p, i, u0);
    q1 = q1 && pred_ok<Sh>(p, i, u1);
  }
  uint64_t a[kMaxKeys] = {0, 0}, b[kMaxKeys] = {0, 0};
#pragma unroll
  for (int i = 0; i < kMaxKeys; ++i) {
    if (i >= Sh::nk(p)) break;
    ld2w(Sh::kw(p, i), p.keys[i].col.ptr, r, a[i], b[i]);
  }
  k0 = pack_key<Sh>(p, a);
  k1 = pack_key<Sh>(p, b);
}

template <class Sh>
__device__ __forceinline__ typename Sh::Key key_one(const Plan& p, int64_t r) {
  uint64_t k[kMaxKeys] = {0, 0};
#pragma unroll
  for (int i = 0; i < kMaxKeys; ++i) {
    if (i >= Sh::nk(p)) break;
    k[i] = ld1w(Sh::kw(p, i), p.keys[i].col.ptr, r);
  }
  return pack_key<Sh>(p, k);
}

template <class Sh>
__device__ __forceinline__ void qk_one(const Plan& p, int64_t r, bool& q, typename Sh::Key& k) {
  q = r < p.n;
  k = 0;
  if (!q) return;
#pragma unroll
  for (int i = 0; i < kMaxPreds; ++i) {
    if (i >= Sh::np(p)) break;
    q = q && pred_ok<Sh>(p, i, ld1w(Sh::pw(p, i), p.preds[i].col.ptr, r));
  }
  k = key_one<Sh>(p, r);
}

// ------------------------------------------------------------------ pass 1: unit and tile summaries
template <class Sh, int K>
__global__ void __launch_bounds__(kSortedThreads) k_sorted_summary(const __grid_constant__ Plan p,
                                                                   const __grid_constant__ SortedArgs a) {
  using Key = typename Sh::Key;
  constexpr int S = 32 * K;
  __shared__ Mono wm[kSortedWarps];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const uint32_t lt = lane_lt();
  const int64_t u = (int64_t)blockIdx.x * kSortedWarps + warp;
  Mono loc = mono_id();
  if (u < a.nunits) {
    const int64_t r0 = u * kSortedUnitRows;
    const int64_t r1 = r0 + kSortedUnitRows < p.n ? r0 + kSortedUnitRows : p.n;
    Key prev_row = r0 > 0 ? key_one<Sh>(p, r0 - 1) : (Key)0;   // sortedness across the unit boundary
    bool has_prev_row = r0 > 0;
    bool has = false, bad = false;
    Key last = 0, first = 0;
    uint32_t heads = 0;
    for (int64_t base = r0; base < r1; base += S) {
      const int64_t rl = base + (int64_t)K * lane;
      bool q[K];
      Key k[K];
      if (base + S <= r1 && p.vec_ok) {
#pragma unroll
        for (int i = 0; i < K / 2; ++i) qk_pair<Sh>(p, rl + 2 * i, q[2 * i], q[2 * i + 1], k[2 * i], k[2 * i + 1]);
      } else {
#pragma unroll
        for (int j = 0; j < K; ++j) qk_one<Sh>(p, rl + j, q[j], k[j]);
      }
      // every row (qualifying or not) must not be smaller than its predecessor
      Key before = __shfl_up_sync(0xffffffffu, k[K - 1], 1);
      if (lane == 0) before = prev_row;
      if (rl < r1 && (lane > 0 || has_prev_row) && k[0] < before) bad = true;
#pragma unroll
      for (int j = 1; j < K; ++j)
        if (rl + j < r1 && k[j] < k[j - 1]) bad = true;
      prev_row = __shfl_sync(0xffffffffu, k[K - 1], 31);
      has_prev_row = true;
      // run starts: compare with the previous qualifying row (lower lanes, else the unit so far)
      bool lq = false;
      Key lk = 0, fk = 0;
#pragma unroll
      for (int j = K - 1; j >= 0; --j)
        if (q[j]) { lq = true; fk = k[j]; }
#pragma unroll
      for (int j = 0; j < K; ++j)
        if (q[j]) lk = k[j];
      const uint32_t QL = __ballot_sync(0xffffffffu, lq);
      if (QL == 0) continue;
      const uint32_t lower = QL & lt;
      const Key from = __shfl_sync(0xffffffffu, lk, lower ? 31 - __clz(lower) : 0);
      bool hv = lower != 0 || has;
      Key pv = lower ? from : last;
      int nh = 0;
#pragma unroll
      for (int j = 0; j < K; ++j)
        if (q[j]) {
          nh += (!hv || k[j] != pv) ? 1 : 0;
          pv = k[j];
          hv = true;
        }
      heads += __reduce_add_sync(0xffffffffu, (unsigned)nh);
      if (!has) first = __shfl_sync(0xffffffffu, fk, __ffs(QL) - 1);
      last = __shfl_sync(0xffffffffu, lk, 31 - __clz(QL));
      has = true;
    }
    if (__any_sync(0xffffffffu, bad) && lane == 0) set_status(p.status, OCL_ERR_INVALID_ARG);
    loc = Mono{heads, (uint64_t)first, (uint64_t)last, has ? 1ULL : 0ULL};
    if (lane == 0) a.sum[u] = loc;
  }
  if (lane == 0) wm[warp] = loc;
  __syncthreads();
  if (warp == 0) {
    const Mono t = mono_warp_reduce(lane < kSortedWarps ? wm[lane] : mono_id(), lane);
    if (lane == 0) a.tile[blockIdx.x] = t;
  }
}

// Exclusive prefix over the tile summaries (in place), one CTA; the total is G.
__global__ void __launch_bounds__(kTileScanThreads) k_sorted_tiles(const __grid_constant__ SortedArgs a) {
  constexpr int PER = 4;
  __shared__ Mono wsm[32];
  __shared__ Mono carry_s;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  if (threadIdx.x == 0) carry_s = mono_id();
  __syncthreads();
  for (int64_t c0 = 0; c0 < a.ntiles; c0 += (int64_t)kTileScanThreads * PER) {
    const int64_t b0 = c0 + (int64_t)threadIdx.x * PER;
    Mono m[PER];
    Mono agg = mono_id();
#pragma unroll
    for (int j = 0; j < PER; ++j) {
      m[j] = b0 + j < a.ntiles ? a.tile[b0 + j] : mono_id();
      agg = mono_combine(agg, m[j]);
    }
    Mono inc = agg;                                             // warp inclusive scan
#pragma unroll
    for (int d = 1; d < 32; d <<= 1) {
      const Mono y = mono_shfl_up(inc, d);
      if (lane >= d) inc = mono_combine(y, inc);
    }
    if (lane == 31) wsm[warp] = inc;
    __syncthreads();
    if (warp == 0) {
      Mono w = wsm[lane];
#pragma unroll
      for (int d = 1; d < 32; d <<= 1) {
        const Mono y = mono_shfl_up(w, d);
        if (lane >= d) w = mono_combine(y, w);
      }
      wsm[lane] = w;
    }
    __syncthreads();
    Mono lex = mono_shfl_up(inc, 1);
    if (lane == 0) lex = mono_id();
    Mono e = mono_combine(carry_s, mono_combine(warp > 0 ? wsm[warp - 1] : mono_id(), lex));
#pragma unroll
    for (int j = 0; j < PER; ++j) {
      if (b0 + j < a.ntiles) a.tile[b0 + j] = e;
      e = mono_combine(e, m[j]);
    }
    __syncthreads();
    if (threadIdx.x == 0) carry_s = mono_combine(carry_s, wsm[31]);
    __syncthreads();
  }
  if (threadIdx.x == 0) {
    const int64_t G = (int64_t)carry_s.runs;
    *a.ngroups_out = G;
    if (G > a.out_capacity) set_status(a.status, OCL_ERR_CAPACITY);
  }
}

// ------------------------------------------------------------------ pass 2: runs -> outputs
// Accumulator of one run piece: count, per value an int128 sum (fp64 values: the
// double's bits in lo) and order-preserving MIN / MAX encodings (0 = identity).
template <int NV>
struct Seg {
  uint32_t cnt;
  I128 s[NV];
  uint64_t mn[NV], mx[NV];
};

template <class Sh, int NV>
__device__ __forceinline__ void seg_zero(const Plan& p, Seg<NV>& a) {
  a.cnt = 0;
#pragma unroll
  for (int v = 0; v < NV; ++v) {
    a.s[v] = I128{0, 0};
    a.mn[v] = a.mx[v] = 0;
  }
}

template <class Sh, int NV>
__device__ __forceinline__ void seg_add(const Plan& p, Seg<NV>& a, const Seg<NV>& b) {
  a.cnt += b.cnt;
#pragma unroll
  for (int v = 0; v < NV; ++v) {
    if (v >= Sh::nv(p)) break;
    if (Sh::fsum(p, v)) {
      if (Sh::vf64(p, v))
        a.s[v].lo = (uint64_t)__double_as_longlong(__dadd_rn(__longlong_as_double((long long)a.s[v].lo),
                                                             __longlong_as_double((long long)b.s[v].lo)));
      else
        a.s[v] = i128_add(a.s[v], b.s[v]);
    }
    if (Sh::fmn(p, v)) a.mn[v] = max(a.mn[v], b.mn[v]);
    if (Sh::fmx(p, v)) a.mx[v] = max(a.mx[v], b.mx[v]);
  }
}

// The run-piece state of one qualifying row.  Rows outside the int64 fast path (and
// fp64 values of a mixed plan) re-read their operands and evaluate exactly.
template <class Sh, int NV, bool F64>
__device__ __forceinline__ void seg_row(const Plan& p, const Row<Sh, NV, F64>& x, int64_t r, Seg<NV>& a) {
  a.cnt = 1;
#pragma unroll
  for (int v = 0; v < NV; ++v) {
    a.s[v] = I128{0, 0};
    a.mn[v] = a.mx[v] = 0;
    if (v >= Sh::nv(p)) break;
    if (Sh::vf64(p, v)) {
      double d;
      if constexpr (F64) {
        d = x.vd[v];
      } else {
        const DevValue& dv = p.vals[v];
        d = value_f64(dv, load_one(dv.a, r), dv.expr >= OCL_EXPR_MUL_1MINUS ? load_one(dv.b, r) : 0,
                      dv.expr >= OCL_EXPR_MUL_1MINUS_1PLUS ? load_one(dv.c, r) : 0);
      }
      a.s[v].lo = (uint64_t)__double_as_longlong(d);
      if (Sh::fmn(p, v)) a.mn[v] = enc_min_f(d);
      if (Sh::fmx(p, v)) a.mx[v] = enc_max_f(d);
    } else {
      I128 e;
      if constexpr (F64) {
        e = I128{0, 0};
      } else {
        if (x.fast) {
          e = i128_from_i64(x.vi[v]);
        } else {
          const DevValue& dv = p.vals[v];
          e = value_i128(dv, load_one(dv.a, r), dv.expr >= OCL_EXPR_MUL_1MINUS ? load_one(dv.b, r) : 0,
                         dv.expr >= OCL_EXPR_MUL_1MINUS_1PLUS ? load_one(dv.c, r) : 0);
        }
      }
      a.s[v] = e;
      if (Sh::fmn(p, v)) a.mn[v] = enc_min_i((int64_t)e.lo);
      if (Sh::fmx(p, v)) a.mx[v] = enc_max_i((int64_t)e.lo);
    }
  }
}

template <class Sh, int NV>
__device__ __forceinline__ void seg_shfl(const Plan& p, Seg<NV>& y, const Seg<NV>& x, int src_delta, bool up) {
  auto sh = [&](uint64_t v) -> uint64_t {
    return up ? __shfl_up_sync(0xffffffffu, v, src_delta) : __shfl_sync(0xffffffffu, v, src_delta);
  };
  y.cnt = up ? __shfl_up_sync(0xffffffffu, x.cnt, src_delta) : __shfl_sync(0xffffffffu, x.cnt, src_delta);
#pragma unroll
  for (int v = 0; v < NV; ++v) {
    y.s[v] = I128{0, 0};
    y.mn[v] = y.mx[v] = 0;
    if (v >= Sh::nv(p)) break;
    if (Sh::fsum(p, v)) {
      y.s[v].lo = sh(x.s[v].lo);
      if (!Sh::vf64(p, v)) y.s[v].hi = sh(x.s[v].hi);
    }
    if (Sh::fmn(p, v)) y.mn[v] = sh(x.mn[v]);
    if (Sh::fmx(p, v)) y.mx[v] = sh(x.mx[v]);
  }
}

// Output row g of a finished run: finalise from registers.
template <class Sh, int NV>
__device__ __forceinline__ void seg_emit(const Plan& p, const FinPlan& f, const Seg<NV>& a, uint64_t key, int64_t g) {
  if (g >= f.out_capacity) return;
  if (f.keys_out) f.keys_out[g] = (int64_t)key;
  for (int i = 0; i < f.naggs; ++i) {
    const OutAgg& o = f.aggs[i];
    if (o.op == OCL_AGG_COUNT) {
      ((int64_t*)o.out)[g] = (int64_t)a.cnt;
      continue;
    }
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      if (v >= Sh::nv(p)) break;
      const DevValue& d = p.vals[v];
      const bool f64 = Sh::vf64(p, v);
      if ((o.op == OCL_AGG_SUM || o.op == OCL_AGG_AVG) && Sh::fsum(p, v) && o.off == d.off_sum) {
        if (o.op == OCL_AGG_SUM) {
          if (f64) ((uint64_t*)o.out)[g] = a.s[v].lo;
          else ((ulonglong2*)o.out)[g] = make_ulonglong2(a.s[v].lo, a.s[v].hi);
        } else {
          const double sum = f64 ? __longlong_as_double((long long)a.s[v].lo) : i128_to_double(a.s[v].lo, a.s[v].hi);
          ((double*)o.out)[g] = __ddiv_rn(sum, __ull2double_rn(a.cnt));
        }
      } else if (o.op == OCL_AGG_MIN && Sh::fmn(p, v) && o.off == d.off_min) {
        if (f64) ((double*)o.out)[g] = dec_min_f(a.mn[v]);
        else ((int64_t*)o.out)[g] = dec_min_i(a.mn[v]);
      } else if (o.op == OCL_AGG_MAX && Sh::fmx(p, v) && o.off == d.off_max) {
        if (f64) ((double*)o.out)[g] = dec_max_f(a.mx[v]);
        else ((int64_t*)o.out)[g] = dec_max_i(a.mx[v]);
      }
    }
  }
}

// Partial row g (ocl_sga_partial layout = the table entry layout with the real key first).
template <class Sh, int NV>
__device__ __forceinline__ void seg_partial(const Plan& p, uint8_t* out, int64_t cap, const Seg<NV>& a, uint64_t key,
                                            int64_t g) {
  if (g >= cap) return;
  uint64_t* row = (uint64_t*)(out + g * (int64_t)p.stride);
  for (int w = 2; w < p.stride / 8; ++w) row[w] = 0;
  row[0] = key;
  row[1] = a.cnt;
#pragma unroll
  for (int v = 0; v < NV; ++v) {
    if (v >= Sh::nv(p)) break;
    const DevValue& d = p.vals[v];
    if (Sh::fsum(p, v)) {
      *(uint64_t*)((uint8_t*)row + d.off_sum) = a.s[v].lo;
      if (!Sh::vf64(p, v)) *(uint64_t*)((uint8_t*)row + d.off_sum + 8) = a.s[v].hi;
    }
    if (Sh::fmn(p, v)) *(uint64_t*)((uint8_t*)row + d.off_min) = a.mn[v];
    if (Sh::fmx(p, v)) *(uint64_t*)((uint8_t*)row + d.off_max) = a.mx[v];
  }
}

// A run piece that may continue across a unit boundary: merge into the chain table
// entry of its group id (find-or-insert by gid, then atomics).
template <class Sh, int NV>
__device__ __forceinline__ void seg_chain(const Plan& p, const SortedArgs& a, const Seg<NV>& s, uint64_t key,
                                          int64_t gid) {
  uint8_t* e = table_find_or_insert(a.chains, a.chain_mask, p.stride, (uint64_t)gid, a.status);
  if (!e) return;
  a.chain_key[(e - a.chains) / p.stride] = key;
  atomicAdd((unsigned long long*)(e + 8), (unsigned long long)s.cnt);
#pragma unroll
  for (int v = 0; v < NV; ++v) {
    if (v >= Sh::nv(p)) break;
    const DevValue& d = p.vals[v];
    if (Sh::fsum(p, v)) {
      if (Sh::vf64(p, v)) atomicAdd((double*)(e + d.off_sum), __longlong_as_double((long long)s.s[v].lo));
      else atomic_add_i128((uint64_t*)(e + d.off_sum), s.s[v].lo, s.s[v].hi);
    }
    if (Sh::fmn(p, v) && s.mn[v]) atomicMax((unsigned long long*)(e + d.off_min), (unsigned long long)s.mn[v]);
    if (Sh::fmx(p, v) && s.mx[v]) atomicMax((unsigned long long*)(e + d.off_max), (unsigned long long)s.mx[v]);
  }
}

// Runs closed during one step, staged per warp (SoA) and written out together.
template <int NV, int S>
struct GenStage {
  uint64_t key[S];
  uint64_t slo[NV][S], shi[NV][S], mn[NV][S], mx[NV][S];
  uint32_t cnt[S];
};
template <int NV, int S>
struct FastStage {
  uint64_t key[S];
  int64_t sum[NV][S];
  uint32_t mn[NV][S], mx[NV][S];
  uint32_t cnt[S];
};
template <int NV, int S>
constexpr size_t stage_bytes() {
  return sizeof(GenStage<NV, S>) > sizeof(FastStage<NV, S>) ? sizeof(GenStage<NV, S>) : sizeof(FastStage<NV, S>);
}

// Selection bitmap of one step (parity-test output): lane l holds rows base + K*l + j.
template <class Sh, int NV, bool F64, int K>
__device__ __forceinline__ void emit_bitmap_k(const Plan& p, int64_t base, int lane, const Row<Sh, NV, F64> (&x)[K]) {
  uint32_t b = 0;
#pragma unroll
  for (int j = 0; j < K; ++j) b |= (uint32_t)x[j].q << j;
  const int64_t words = (p.n + 31) >> 5;
#pragma unroll
  for (int w = 0; w < K; ++w) {
    const uint32_t v = __reduce_or_sync(0xffffffffu, ((K * lane) >> 5) == w ? b << ((K * lane) & 31) : 0u);
    const int64_t wi = (base >> 5) + w;
    if (lane == w && wi < words) p.bitmap_out[wi] = v;
  }
}

// Accumulator policies of a step.  GenOps: any plan (Seg: int128 sums, 64-bit MIN /
// MAX encodings).  FastOps: integer COL values when every qualifying row of the step
// fits int32 (the common case): int64 sums (a unit holds 2^11 rows), 32-bit
// encodings, fewer shuffles and adds, and a direct output map.
template <class Sh, int NV, bool F64, int S>
struct GenOps {
  using T = Seg<NV>;
  using Stg = GenStage<NV, S>;
  static __device__ __forceinline__ void zero(const Plan& p, T& a) { seg_zero<Sh, NV>(p, a); }
  static __device__ __forceinline__ void add(const Plan& p, T& a, const T& b) { seg_add<Sh, NV>(p, a, b); }
  static __device__ __forceinline__ void row(const Plan& p, const Row<Sh, NV, F64>& x, int64_t r, T& a) {
    if (x.q) seg_row<Sh, NV, F64>(p, x, r, a);
    else seg_zero<Sh, NV>(p, a);
  }
  static __device__ __forceinline__ void shfl(const Plan& p, T& y, const T& x, int d, bool up) {
    seg_shfl<Sh, NV>(p, y, x, d, up);
  }
  static __device__ __forceinline__ void gen(const Plan& p, const T& a, Seg<NV>& g) { g = a; }
  static __device__ __forceinline__ void put(const Plan& p, Stg& st, int slot, const T& s, uint64_t key) {
    st.key[slot] = key;
    st.cnt[slot] = s.cnt;
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      if (v >= Sh::nv(p)) break;
      if (Sh::fsum(p, v)) {
        st.slo[v][slot] = s.s[v].lo;
        if (!Sh::vf64(p, v)) st.shi[v][slot] = s.s[v].hi;
      }
      if (Sh::fmn(p, v)) st.mn[v][slot] = s.mn[v];
      if (Sh::fmx(p, v)) st.mx[v][slot] = s.mx[v];
    }
  }
  static __device__ __forceinline__ void get(const Plan& p, const Stg& st, int slot, Seg<NV>& s, uint64_t& key) {
    seg_zero<Sh, NV>(p, s);
    key = st.key[slot];
    s.cnt = st.cnt[slot];
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      if (v >= Sh::nv(p)) break;
      if (Sh::fsum(p, v)) {
        s.s[v].lo = st.slo[v][slot];
        if (!Sh::vf64(p, v)) s.s[v].hi = st.shi[v][slot];
      }
      if (Sh::fmn(p, v)) s.mn[v] = st.mn[v][slot];
      if (Sh::fmx(p, v)) s.mx[v] = st.mx[v][slot];
    }
  }
  static __device__ __forceinline__ void emit(const Plan& p, const SortedArgs& a, const Stg& st, int slot, int64_t g) {
    Seg<NV> s;
    uint64_t key;
    get(p, st, slot, s, key);
    if (a.partial_out) seg_partial<Sh, NV>(p, a.partial_out, a.out_capacity, s, key, g);
    else seg_emit<Sh, NV>(p, a.fin, s, key, g);
  }
};

template <int NV>
struct FastSeg {
  uint32_t cnt;
  int64_t sum[NV];
  uint32_t mn[NV], mx[NV];    // enc32 encodings (0 = identity)
};

template <class Sh, int NV, bool F64, int S>
struct FastOps {
  using T = FastSeg<NV>;
  using Stg = FastStage<NV, S>;
  static __device__ __forceinline__ void zero(const Plan& p, T& a) {
    a.cnt = 0;
#pragma unroll
    for (int v = 0; v < NV; ++v) { a.sum[v] = 0; a.mn[v] = a.mx[v] = 0; }
  }
  static __device__ __forceinline__ void add(const Plan& p, T& a, const T& b) {
    a.cnt += b.cnt;
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      if (Sh::fsum(p, v)) a.sum[v] += b.sum[v];
      if (Sh::fmn(p, v)) a.mn[v] = max(a.mn[v], b.mn[v]);
      if (Sh::fmx(p, v)) a.mx[v] = max(a.mx[v], b.mx[v]);
    }
  }
  static __device__ __forceinline__ void row(const Plan& p, const Row<Sh, NV, F64>& x, int64_t, T& a) {
    a.cnt = x.q ? 1u : 0u;
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      const int32_t w = (int32_t)x.vi[v];
      a.sum[v] = x.q ? (int64_t)w : 0;
      a.mn[v] = (Sh::fmn(p, v) && x.q) ? enc32_min(w) : 0u;
      a.mx[v] = (Sh::fmx(p, v) && x.q) ? enc32_max(w) : 0u;
    }
  }
  static __device__ __forceinline__ void shfl(const Plan& p, T& y, const T& x, int d, bool up) {
    y.cnt = up ? __shfl_up_sync(0xffffffffu, x.cnt, d) : __shfl_sync(0xffffffffu, x.cnt, d);
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      y.sum[v] = 0;
      y.mn[v] = y.mx[v] = 0;
      if (Sh::fsum(p, v))
        y.sum[v] = up ? __shfl_up_sync(0xffffffffu, x.sum[v], d) : __shfl_sync(0xffffffffu, x.sum[v], d);
      if (Sh::fmn(p, v)) y.mn[v] = up ? __shfl_up_sync(0xffffffffu, x.mn[v], d) : __shfl_sync(0xffffffffu, x.mn[v], d);
      if (Sh::fmx(p, v)) y.mx[v] = up ? __shfl_up_sync(0xffffffffu, x.mx[v], d) : __shfl_sync(0xffffffffu, x.mx[v], d);
    }
  }
  static __device__ __forceinline__ void gen(const Plan& p, const T& a, Seg<NV>& g) {
    g.cnt = a.cnt;
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      g.s[v] = i128_from_i64(a.sum[v]);
      g.mn[v] = (Sh::fmn(p, v) && a.cnt) ? enc_min_i((int32_t)(~a.mn[v] ^ 0x80000000u)) : 0;
      g.mx[v] = (Sh::fmx(p, v) && a.cnt) ? enc_max_i((int32_t)(a.mx[v] ^ 0x80000000u)) : 0;
    }
  }
  // Seg -> FastSeg when it fits (sums in int64, MIN / MAX in int32)
  static __device__ __forceinline__ bool from_gen(const Plan& p, const Seg<NV>& g, T& a) {
    bool ok = true;
    a.cnt = g.cnt;
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      a.sum[v] = (int64_t)g.s[v].lo;
      ok = ok && g.s[v].hi == (uint64_t)((int64_t)g.s[v].lo >> 63);
      a.mn[v] = a.mx[v] = 0;
      if (Sh::fmn(p, v) && g.cnt) {
        const int64_t m = dec_min_i(g.mn[v]);
        ok = ok && fits_i32(m);
        a.mn[v] = enc32_min((int32_t)m);
      }
      if (Sh::fmx(p, v) && g.cnt) {
        const int64_t m = dec_max_i(g.mx[v]);
        ok = ok && fits_i32(m);
        a.mx[v] = enc32_max((int32_t)m);
      }
    }
    return ok;
  }
  static __device__ __forceinline__ void put(const Plan& p, Stg& st, int slot, const T& s, uint64_t key) {
    st.key[slot] = key;
    st.cnt[slot] = s.cnt;
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      if (Sh::fsum(p, v)) st.sum[v][slot] = s.sum[v];
      if (Sh::fmn(p, v)) st.mn[v][slot] = s.mn[v];
      if (Sh::fmx(p, v)) st.mx[v][slot] = s.mx[v];
    }
  }
  static __device__ __forceinline__ void get(const Plan& p, const Stg& st, int slot, Seg<NV>& s, uint64_t& key) {
    T f;
    key = st.key[slot];
    f.cnt = st.cnt[slot];
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      f.sum[v] = Sh::fsum(p, v) ? st.sum[v][slot] : 0;
      f.mn[v] = Sh::fmn(p, v) ? st.mn[v][slot] : 0u;
      f.mx[v] = Sh::fmx(p, v) ? st.mx[v][slot] : 0u;
    }
    gen(p, f, s);
  }
  static __device__ __forceinline__ void emit(const Plan& p, const SortedArgs& a, const Stg& st, int slot, int64_t g) {
    if (!a.fe.ok) {
      Seg<NV> s;
      uint64_t key;
      get(p, st, slot, s, key);
      if (a.partial_out) seg_partial<Sh, NV>(p, a.partial_out, a.out_capacity, s, key, g);
      else seg_emit<Sh, NV>(p, a.fin, s, key, g);
      return;
    }
    if (g >= a.fin.out_capacity) return;
    const uint32_t c = st.cnt[slot];
    if (a.fin.keys_out) a.fin.keys_out[g] = (int64_t)st.key[slot];
    if (a.fe.cnt) a.fe.cnt[g] = (int64_t)c;
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      if (Sh::fsum(p, v)) {
        const int64_t sm = st.sum[v][slot];
        if (a.fe.sum[v]) ((ulonglong2*)a.fe.sum[v])[g] = make_ulonglong2((uint64_t)sm, (uint64_t)(sm >> 63));
        if (a.fe.avg[v]) a.fe.avg[v][g] = __ddiv_rn(__ll2double_rn(sm), __ull2double_rn(c));
      }
      if (Sh::fmn(p, v) && a.fe.mn[v]) a.fe.mn[v][g] = (int32_t)(~st.mn[v][slot] ^ 0x80000000u);
      if (Sh::fmx(p, v) && a.fe.mx[v]) a.fe.mx[v][g] = (int32_t)(st.mx[v][slot] ^ 0x80000000u);
    }
  }
};

// The state of one unit's pass.
template <class Sh, int NV, int S>
struct UnitCtx {
  const Plan& p;
  const SortedArgs& a;
  uint8_t* stage;
  int64_t gbase, last_idx, seg_count;
  int lane;
  uint32_t lt;
};

// One step with policy Ops: lane fold, warp segmented scan over the lanes' open pieces,
// runs closed in the step staged and written as one range of output rows; the unit's
// first / last run goes to the chain table instead.  carry: the run open before and
// after the step.
template <class Ops, class Sh, int NV, bool F64, int K, int S>
__device__ __forceinline__ void step_runs(UnitCtx<Sh, NV, S>& c, const Row<Sh, NV, F64> (&x)[K], int64_t rl,
                                          uint32_t hbits, int nh, int heads_before, int heads_step,
                                          typename Sh::Key pk, typename Ops::T& carry) {
  using T = typename Ops::T;
  const Plan& p = c.p;
  typename Ops::Stg& st = *(typename Ops::Stg*)c.stage;
  const int64_t slot0 = c.seg_count - 1;                       // run index of staging slot 0
  // lane-local fold: P1 = rows before the lane's first run start (continuing from the
  // left), runs closed inside the lane (staged), cur = the open piece
  T cur, P1;
  Ops::zero(p, cur);
  Ops::zero(p, P1);
  typename Sh::Key curkey = pk;
  int slot = (int)(c.seg_count + heads_before - 1 - slot0);     // slot of the run a lane start closes
#pragma unroll
  for (int j = 0; j < K; ++j) {
    T row;
    Ops::row(p, x[j], rl + j, row);
    if ((hbits >> j) & 1u) {
      if (j > 0 && (hbits & ((1u << j) - 1u))) Ops::put(p, st, slot, cur, (uint64_t)curkey);
      else P1 = cur;
      ++slot;
      cur = row;
      curkey = x[j].key;
    } else {
      Ops::add(p, cur, row);
    }
  }
  // segmented inclusive scan of the open pieces; segments start at lanes with a run start
  const uint32_t F = __ballot_sync(0xffffffffu, nh > 0);
  const uint32_t upto = F & (c.lt | (1u << c.lane));
  const int sstart = upto ? 31 - __clz(upto) : 0;
  T Sc = cur;
#pragma unroll
  for (int d = 1; d < 32; d <<= 1) {
    T y;
    Ops::shfl(p, y, Sc, d, true);
    if (c.lane - d >= sstart) Ops::add(p, Sc, y);
  }
  T E;                                                         // inclusive scan of the lane before
  Ops::shfl(p, E, Sc, 1, true);
  if (nh > 0 && c.seg_count + heads_before - 1 >= 0) {         // the run ending before the lane's first start
    if (c.lane > 0) Ops::add(p, P1, E);
    if ((F & c.lt) == 0) Ops::add(p, P1, carry);
    Ops::put(p, st, (int)(c.seg_count + heads_before - 1 - slot0), P1, (uint64_t)pk);
  }
  T open;
  Ops::shfl(p, open, Sc, 31, false);
  if (F) carry = open;
  else Ops::add(p, carry, open);
  __syncwarp();
  for (int s = c.lane; s < heads_step; s += 32) {              // write the runs closed in this step
    const int64_t idx = slot0 + s;
    if (idx < 0) continue;
    if (idx == 0 || idx == c.last_idx) {
      Seg<NV> g;
      uint64_t key;
      Ops::get(p, st, s, g, key);
      seg_chain<Sh, NV>(p, c.a, g, key, c.gbase + idx);
    } else {
      Ops::emit(p, c.a, st, s, c.gbase + idx);
    }
  }
  __syncwarp();
  c.seg_count += heads_step;
}

template <class Sh>
constexpr bool fast_capable() {
  if constexpr (Sh::kStatic) return Sh::all_int_cols();
  else return false;
}

template <class Sh, int NV, bool F64, int K>
__global__ void __launch_bounds__(kSortedThreads) k_sorted_agg(const __grid_constant__ Plan p,
                                                               const __grid_constant__ SortedArgs a) {
  using Key = typename Sh::Key;
  constexpr int S = 32 * K;                                    // rows (and at most runs) per step
  constexpr bool FAST = fast_capable<Sh>();
  using GO = GenOps<Sh, NV, F64, S>;
  using FO = FastOps<Sh, NV, F64, S>;
  extern __shared__ __align__(16) uint8_t sm_raw[];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const int64_t u = (int64_t)blockIdx.x * kSortedWarps + warp;
  if (u >= a.nunits) return;
  const Mono us = a.sum[u];
  const int64_t r0 = u * kSortedUnitRows;
  const int64_t r1 = r0 + kSortedUnitRows < p.n ? r0 + kSortedUnitRows : p.n;
  if (!us.has) {
    if (p.bitmap_out) {                                        // parity-test output only
      const int64_t words = (p.n + 31) >> 5;
      for (int64_t w = (r0 >> 5) + lane; w < ((r1 + 31) >> 5) && w < words; w += 32) p.bitmap_out[w] = 0u;
    }
    return;
  }
  // prefix of the unit = tile prefix + the earlier units of the tile
  const Mono before = mono_warp_reduce(lane < warp ? a.sum[(int64_t)blockIdx.x * kSortedWarps + lane] : mono_id(), lane);
  const Mono E0 = mono_combine(a.tile[blockIdx.x], before);
  const bool cin = E0.has && E0.last == us.first;
  const uint32_t lt = lane_lt();
  UnitCtx<Sh, NV, S> c{p, a, sm_raw + (size_t)warp * stage_bytes<NV, S>(), (int64_t)E0.runs - (cin ? 1 : 0),
                       (int64_t)us.runs - 1, 0, lane, lt};
  typename GO::T carry_g;
  typename FO::T carry_f;
  GO::zero(p, carry_g);
  FO::zero(p, carry_f);
  bool carry_fast = true, has_carry = false;
  Key carry_key = 0;
  for (int64_t base = r0; base < r1; base += S) {
    Row<Sh, NV, F64> x[K];
    const int64_t rl = base + (int64_t)K * lane;
    if (base + S <= r1 && p.vec_ok) {
#pragma unroll
      for (int i = 0; i < K / 2; ++i) eval_pair<Sh, NV, F64>(p, rl + 2 * i, x[2 * i], x[2 * i + 1]);
    } else {
#pragma unroll
      for (int j = 0; j < K; ++j) eval_one<Sh, NV, F64>(p, rl + j, x[j]);
    }
    if (p.bitmap_out) emit_bitmap_k<Sh, NV, F64, K>(p, base, lane, x);
    bool lq = false, lfast = true;
    Key lk = 0;
#pragma unroll
    for (int j = 0; j < K; ++j)
      if (x[j].q) { lq = true; lk = x[j].key; lfast = lfast && x[j].fast; }
    const uint32_t QL = __ballot_sync(0xffffffffu, lq);
    if (QL == 0) continue;                                     // warp-uniform
    const uint32_t lower = QL & lt;
    const Key from = __shfl_sync(0xffffffffu, lk, lower ? 31 - __clz(lower) : 0);
    const bool hp = lower != 0 || has_carry;
    const Key pk = lower ? from : carry_key;                   // previous qualifying key of the lane's rows
    uint32_t hbits = 0;                                        // run starts among the lane's rows
    {
      Key pv = pk;
      bool hv = hp;
#pragma unroll
      for (int j = 0; j < K; ++j)
        if (x[j].q) {
          if (!hv || x[j].key != pv) hbits |= 1u << j;
          pv = x[j].key;
          hv = true;
        }
    }
    const int nh = __popc(hbits);
    int hb_incl = nh;                                          // warp prefix sum of run starts
#pragma unroll
    for (int d = 1; d < 32; d <<= 1) {
      const int y = __shfl_up_sync(0xffffffffu, hb_incl, d);
      if (lane >= d) hb_incl += y;
    }
    const int heads_step = __shfl_sync(0xffffffffu, hb_incl, 31);
    bool fast_step = false;
    if constexpr (FAST) fast_step = carry_fast && __all_sync(0xffffffffu, lfast);
    if (fast_step) {
      if constexpr (FAST) step_runs<FO, Sh, NV, F64, K, S>(c, x, rl, hbits, nh, hb_incl - nh, heads_step, pk, carry_f);
    } else {
      if constexpr (FAST) {
        if (carry_fast) FO::gen(p, carry_f, carry_g);
      }
      step_runs<GO, Sh, NV, F64, K, S>(c, x, rl, hbits, nh, hb_incl - nh, heads_step, pk, carry_g);
      if constexpr (FAST) carry_fast = FO::from_gen(p, carry_g, carry_f);
    }
    carry_key = __shfl_sync(0xffffffffu, lk, 31 - __clz(QL));
    has_carry = true;
  }
  if (lane == 0 && c.seg_count > 0) {                          // the unit's last run: chain table
    if (carry_fast && FAST) FO::gen(p, carry_f, carry_g);
    seg_chain<Sh, NV>(p, a, carry_g, (uint64_t)carry_key, c.gbase + c.seg_count - 1);
  }
}

__global__ void k_sorted_chain_emit(const uint8_t* chains, int32_t stride, const uint64_t* chain_key, uint64_t cap,
                                    const __grid_constant__ FinPlan f, uint8_t* partial_out, int64_t out_capacity) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < cap; i += (uint64_t)gridDim.x * blockDim.x) {
    const uint8_t* e = chains + i * (uint64_t)stride;
    const uint64_t sk = *(const uint64_t*)e;
    if (!sk) continue;
    const int64_t g = (int64_t)~sk;
    if (!partial_out) {
      emit_final(f, e, chain_key[i], g);
    } else if (g < out_capacity) {                            // partial row: the entry with the real key first
      uint64_t* row = (uint64_t*)(partial_out + g * (int64_t)stride);
      row[0] = chain_key[i];
      for (int w = 1; w < stride / 8; ++w) row[w] = ((const uint64_t*)e)[w];
    }
  }
}

// ------------------------------------------------------------------ unfused sorted group build
constexpr int kGbsRounds = 8;                                   // 32-row chunks per warp per tile
constexpr int kGbsTileRows = kSortedWarps * kGbsRounds * 32;    // 2048
constexpr uint64_t kGbsAgg = 1ULL << 62, kGbsIncl = 2ULL << 62, kGbsVal = (1ULL << 62) - 1;

__device__ __forceinline__ uint64_t gbs_ld_acquire(const uint64_t* p) {
  uint64_t v;
  asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void gbs_st_release(uint64_t* p, uint64_t v) {
  asm volatile("st.release.gpu.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}

__device__ __forceinline__ uint64_t gbs_key(const Plan& p, int64_t j) {
  const int64_t r = p.oids ? (int64_t)p.oids[j] : j;
  return row_key_scalar(p, r);
}

__global__ void __launch_bounds__(kSortedThreads) k_group_build_sorted(const __grid_constant__ Plan p, int32_t* gid_out,
                                                                       int64_t* keys_out, int64_t out_capacity,
                                                                       int64_t* ngroups, unsigned long long* counter,
                                                                       uint64_t* tstat, int64_t ntiles) {
  __shared__ uint32_t warp_tot[kSortedWarps];
  __shared__ uint64_t sh_tile, sh_excl;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const int64_t m = p.m_dev ? (*p.m_dev < p.n ? *p.m_dev : p.n) : p.n;
  for (;;) {
    if (threadIdx.x == 0) sh_tile = atomicAdd(counter, 1ULL);
    __syncthreads();
    const int64_t tile = (int64_t)sh_tile;
    if (tile >= ntiles) break;
    const int64_t j0 = tile * kGbsTileRows + (int64_t)warp * kGbsRounds * 32;
    uint32_t hm[kGbsRounds];
    uint64_t key[kGbsRounds];
    uint32_t tot = 0;
    bool bad = false;
#pragma unroll
    for (int i = 0; i < kGbsRounds; ++i) {
      const int64_t j = j0 + 32 * i + lane;
      bool head = false;
      key[i] = 0;
      if (j < m) {
        key[i] = gbs_key(p, j);
        const uint64_t prev = j > 0 ? gbs_key(p, j - 1) : 0;   // predecessor (mostly an L1 hit)
        head = j == 0 || key[i] != prev;
        bad |= j > 0 && key[i] < prev;
      }
      hm[i] = __ballot_sync(0xffffffffu, head);
      tot += __popc(hm[i]);
    }
    if (__any_sync(0xffffffffu, bad) && lane == 0) set_status(p.status, OCL_ERR_INVALID_ARG);
    if (lane == 0) warp_tot[warp] = tot;
    __syncthreads();
    uint32_t warp_base = 0, tile_agg = 0;
#pragma unroll
    for (int w = 0; w < kSortedWarps; ++w) {
      warp_base += w < warp ? warp_tot[w] : 0;
      tile_agg += warp_tot[w];
    }
    if (warp == 0) {                                 // decoupled look-back over tile head counts
      uint64_t excl = 0;
      if (tile == 0) {
        if (lane == 0) gbs_st_release(tstat, kGbsIncl | tile_agg);
      } else {
        if (lane == 0) gbs_st_release(tstat + tile, kGbsAgg | tile_agg);
        int64_t pos = tile - 1;
        for (;;) {
          const int64_t idx = pos - lane;
          uint64_t s = kGbsIncl;
          if (idx >= 0) {
            do { s = gbs_ld_acquire(tstat + idx); } while ((s >> 62) == 0);
          }
          const uint32_t incl = __ballot_sync(0xffffffffu, (s >> 62) == 2);
          const int first = incl ? __ffs(incl) - 1 : 32;
          uint64_t c = lane <= first ? (s & kGbsVal) : 0;
          for (int o = 16; o > 0; o >>= 1) c += __shfl_xor_sync(0xffffffffu, c, o);
          excl += c;
          if (first < 32) break;
          pos -= 32;
        }
        if (lane == 0) gbs_st_release(tstat + tile, kGbsIncl | (excl + tile_agg));
      }
      if (lane == 0) {
        sh_excl = excl;
        if (tile == ntiles - 1) {
          *ngroups = (int64_t)(excl + tile_agg);
          if ((int64_t)(excl + tile_agg) > out_capacity) set_status(p.status, OCL_ERR_CAPACITY);
        }
      }
    }
    __syncthreads();
    uint64_t before = sh_excl + warp_base;           // heads before this warp's rows
#pragma unroll
    for (int i = 0; i < kGbsRounds; ++i) {
      const int64_t j = j0 + 32 * i + lane;
      const int64_t g = (int64_t)before + __popc(hm[i] & ((2u << lane) - 1)) - 1;   // heads <= j, minus 1
      if (j < m) {
        gid_out[j] = (int32_t)g;
        if (((hm[i] >> lane) & 1u) && keys_out && g < out_capacity) keys_out[g] = (int64_t)key[i];
      }
      before += __popc(hm[i]);
    }
    __syncthreads();
  }
}

// ------------------------------------------------------------------ host side
namespace {
constexpr size_t al256(size_t x) { return (x + 255) / 256 * 256; }
int64_t sorted_units(const Plan& p) { return (p.n + kSortedUnitRows - 1) / kSortedUnitRows; }
int64_t sorted_tiles(const Plan& p) { return (p.n + kSortedTileRows - 1) / kSortedTileRows; }
uint64_t chain_cap(int64_t nunits) {
  uint64_t c = 64;
  while (c < 4 * (uint64_t)nunits) c <<= 1;                     // <= 2 chain pieces per unit: load <= 1/2
  return c;
}
size_t chain_bytes(const Plan& p) { return al256((chain_cap(sorted_units(p)) + 1) * (size_t)p.stride); }

// Direct output map of the fast path (integer COL values): one pointer per output kind.
FastEmit build_fast_emit(const Plan& p, const FinPlan& f) {
  FastEmit e;
  memset(&e, 0, sizeof(e));
  e.ok = 1;
  auto set = [&](auto*& slot, void* ptr) {
    if (slot) e.ok = 0;                                           // the same output twice: generic emission
    slot = (decltype(slot))ptr;
  };
  for (int i = 0; i < f.naggs; ++i) {
    const OutAgg& o = f.aggs[i];
    if (o.op == OCL_AGG_COUNT) { set(e.cnt, o.out); continue; }
    bool found = false;
    for (int v = 0; v < p.nvals && !found; ++v) {
      const DevValue& d = p.vals[v];
      if (d.is_f64 || d.expr != OCL_EXPR_COL) { e.ok = 0; break; }
      if ((o.op == OCL_AGG_SUM || o.op == OCL_AGG_AVG) && o.off == d.off_sum) {
        if (o.op == OCL_AGG_SUM) set(e.sum[v], o.out);
        else set(e.avg[v], o.out);
        found = true;
      } else if (o.op == OCL_AGG_MIN && o.off == d.off_min) {
        set(e.mn[v], o.out);
        found = true;
      } else if (o.op == OCL_AGG_MAX && o.off == d.off_max) {
        set(e.mx[v], o.out);
        found = true;
      }
    }
    if (!found) e.ok = 0;
  }
  return e;
}
}  // namespace

size_t sorted_ws_bytes(const Plan& p) {
  const int64_t nu = sorted_units(p), nt = sorted_tiles(p);
  return chain_bytes(p) + al256(nu * sizeof(Mono)) + al256(nt * sizeof(Mono)) +
         al256((chain_cap(nu) + 1) * 8) + 256;
}

template <class Sh, int NV, bool F64, int K>
static cudaError_t sorted_run(const Plan& p, const SortedArgs& a, int sms, cudaStream_t s) {
  const int grid = (int)a.ntiles;
  count_launch(4);
  k_sorted_summary<Sh, 4><<<grid, kSortedThreads, 0, s>>>(p, a);
  k_sorted_tiles<<<1, kTileScanThreads, 0, s>>>(a);
  const size_t smem = (size_t)kSortedWarps * stage_bytes<NV, 32 * K>();
  auto fn = k_sorted_agg<Sh, NV, F64, K>;
  cudaError_t e = cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  if (e != cudaSuccess) return e;
  e = cudaFuncSetAttribute(fn, cudaFuncAttributePreferredSharedMemoryCarveout, 100);
  if (e != cudaSuccess) return e;
  fn<<<grid, kSortedThreads, smem, s>>>(p, a);
  const uint64_t cap = a.chain_mask + 1;
  const int cgrid = (int)std::min<uint64_t>((cap + 255) / 256, (uint64_t)sms * 4);
  k_sorted_chain_emit<<<cgrid, 256, 0, s>>>(a.chains, p.stride, a.chain_key, cap, a.fin, a.partial_out,
                                            a.out_capacity);
  return cudaGetLastError();
}

template <bool F64>
static cudaError_t sorted_dyn(const Plan& p, const SortedArgs& a, int sms, cudaStream_t s) {
  if (p.nvals <= 1) return sorted_run<DynShape, 1, F64, 2>(p, a, sms, s);
  if (p.nvals <= 2) return sorted_run<DynShape, 2, F64, 2>(p, a, sms, s);
  if (p.nvals <= 4) return sorted_run<DynShape, 4, F64, 2>(p, a, sms, s);
  return sorted_run<DynShape, 6, F64, 2>(p, a, sms, s);
}

cudaError_t launch_sorted(const Plan& p, const FinPlan& fin, bool values_f64, void* ws, int32_t* status,
                          int64_t* ngroups_out, int64_t out_capacity, int sms, cudaStream_t s, int* kind,
                          uint8_t* partial_out) {
  *kind = 40;
  if (p.n == 0) return cudaMemsetAsync(ngroups_out, 0, 8, s);
  SortedArgs a;
  memset(&a, 0, sizeof(a));
  a.nunits = sorted_units(p);
  a.ntiles = sorted_tiles(p);
  const uint64_t cap = chain_cap(a.nunits);
  uint8_t* w = (uint8_t*)ws;
  cudaError_t e = cudaMemsetAsync(w, 0, chain_bytes(p), s);      // empty chain table
  if (e != cudaSuccess) return e;
  a.chains = w;
  w += chain_bytes(p);
  a.sum = (Mono*)w;
  w += al256(a.nunits * sizeof(Mono));
  a.tile = (Mono*)w;
  w += al256(a.ntiles * sizeof(Mono));
  a.chain_key = (uint64_t*)w;
  a.chain_mask = cap - 1;
  a.ngroups_out = ngroups_out;
  a.out_capacity = out_capacity;
  a.status = status;
  a.fin = fin;
  a.fe = build_fast_emit(p, fin);
  a.partial_out = partial_out;
  if (partial_out) a.fe.ok = 0;                               // partial rows: the generic row writer
  if (p.vec_ok && shape_match<ShK64>(p)) {
    *kind = 41;
    const char* ek = getenv("OCL_SORTED_K");               // tuning knob: rows per lane per step
    const int K = ek ? atoi(ek) : 8;
    if (K == 2) return sorted_run<ShK64, 1, false, 2>(p, a, sms, s);
    if (K == 4) return sorted_run<ShK64, 1, false, 4>(p, a, sms, s);
    return sorted_run<ShK64, 1, false, 8>(p, a, sms, s);
  }
  if (p.vec_ok && shape_match<ShP32K64>(p)) {
    *kind = 42;
    return sorted_run<ShP32K64, 1, false, 8>(p, a, sms, s);
  }
  return values_f64 ? sorted_dyn<true>(p, a, sms, s) : sorted_dyn<false>(p, a, sms, s);
}

size_t group_build_sorted_ws_bytes(int64_t max_rows) {
  const int64_t nt = (max_rows + kGbsTileRows - 1) / kGbsTileRows;
  return 256 + (size_t)nt * 8;
}

cudaError_t launch_group_build_sorted(const Plan& p, int32_t* gid_out, int64_t* keys_out, int64_t out_capacity,
                                      int64_t* ngroups, void* ws, int sms, cudaStream_t s) {
  cudaError_t e = cudaMemsetAsync(ngroups, 0, 8, s);
  if (e != cudaSuccess || p.n == 0) return e;
  const int64_t nt = (p.n + kGbsTileRows - 1) / kGbsTileRows;
  e = cudaMemsetAsync(ws, 0, group_build_sorted_ws_bytes(p.n), s);
  if (e != cudaSuccess) return e;
  int64_t grid = (int64_t)sms * 4;
  if (nt < grid) grid = nt;
  count_launch();
  k_group_build_sorted<<<(int)grid, kSortedThreads, 0, s>>>(p, gid_out, keys_out, out_capacity, ngroups,
                                                            (unsigned long long*)ws, (uint64_t*)((uint8_t*)ws + 256), nt);
  return cudaGetLastError();
}

}  // namespace ocl
