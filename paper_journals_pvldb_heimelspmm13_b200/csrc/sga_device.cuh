// sga_device.cuh — device building blocks of the fused select -> group -> aggregate
// kernel (fused.cu) and of the grouped aggregation over group ids (aggregate.cu):
// plan shapes, row evaluation, the private-slot / CTA-table / warp-aggregated HBM
// accumulation tiers.  See fused.cu for the design notes and paper citations.
#pragma once

#ifndef OCL_VAR_FITS
#define OCL_VAR_FITS 0
#endif
#ifndef OCL_VAR_PIPE
#define OCL_VAR_PIPE 1
#endif

#include <type_traits>

#include "launch.cuh"
#include "rowops.cuh"

namespace ocl {

constexpr int kFusedThreads = 256;
constexpr int kRegSlots = 4;
constexpr int kUnits = 2;
constexpr int kTileRows = 64 * kUnits;

// ------------------------------------------------------------------ shapes
enum : uint32_t { VF_SUM = 1, VF_MIN = 2, VF_MAX = 4 };
// value descriptor: kind (2 bits) | a (3) | b (3) | c (3) | flags (3)
__host__ __device__ constexpr uint32_t vop(uint32_t kind, uint32_t flags, uint32_t a, uint32_t b = 0,
                                           uint32_t c = 0) {
  return kind | (a << 2) | (b << 5) | (c << 8) | (flags << 11);
}

struct DynShape {
  static constexpr bool kStatic = false;
  static constexpr bool kCta = true;       // the CTA table may be used (decided at run time by smem_cap)
  static constexpr int NC = 1;
  using Key = uint64_t;
  __device__ static int np(const Plan& p) { return p.npreds; }
  __device__ static int pw(const Plan& p, int i) { return p.preds[i].col.width; }
  __device__ static bool pf64(const Plan& p, int i) { return p.preds[i].is_f64; }
  __device__ static int nk(const Plan& p) { return p.nkeys; }
  __device__ static int kw(const Plan& p, int i) { return p.keys[i].col.width; }
  __device__ static uint64_t kmask(const Plan& p, int i) { return p.keys[i].mask; }
  __device__ static int kshift(const Plan& p, int i) { return p.keys[i].shift; }
  __device__ static int nv(const Plan& p) { return p.nvals; }
  __device__ static int kind(const Plan& p, int v) { return p.vals[v].expr; }
  __device__ static bool fsum(const Plan& p, int v) { return p.vals[v].off_sum >= 0; }
  __device__ static bool fmn(const Plan& p, int v) { return p.vals[v].off_min >= 0; }
  __device__ static bool fmx(const Plan& p, int v) { return p.vals[v].off_max >= 0; }
  __device__ static bool vf64(const Plan& p, int v) { return p.vals[v].is_f64; }
  __device__ static bool special(uint64_t k) { return k == ~0ULL; }
  __device__ static int po_sum(const Plan& p, int v) { return p.vals[v].po_sum; }
  __device__ static int po_hi(const Plan& p, int v) { return p.vals[v].po_hi; }
  __device__ static int po_min(const Plan& p, int v) { return p.vals[v].po_min; }
  __device__ static int po_max(const Plan& p, int v) { return p.vals[v].po_max; }
  __device__ static int rec(const Plan& p) { return p.priv_rec; }
};

// PW: predicate width (0 = none); K0W/K1W: key widths (0 = absent); NC distinct
// 8-byte value columns (int64, or fp64 when F64); OPS: vop(...) per value.
template <int PW, bool PF64, int K0W, int K1W, int NC_, bool F64, uint32_t... OPS>
struct StaticShape {
  static constexpr bool kStatic = true;
  static constexpr int NC = NC_;
  static constexpr int KBITS = 8 * (K0W + K1W);
  using Key = typename std::conditional<(KBITS > 0 && KBITS <= 32), uint32_t, uint64_t>::type;
  static constexpr int NVS = sizeof...(OPS);
  __host__ __device__ static constexpr uint32_t op(int v) {
    const uint32_t a[NVS] = {OPS...};
    return a[v];
  }
  __host__ __device__ static constexpr bool all_int_cols() {
    for (int v = 0; v < NVS; ++v)
      if ((op(v) & 3) != 0) return false;
    return !F64;
  }
  static constexpr bool kCta = all_int_cols();   // the CTA table holds int32 COL values only
  __host__ __device__ static constexpr int np(const Plan&) { return PW ? 1 : 0; }
  __host__ __device__ static constexpr int pw(const Plan&, int) { return PW; }
  __host__ __device__ static constexpr bool pf64(const Plan&, int) { return PF64; }
  __host__ __device__ static constexpr int nk(const Plan&) { return (K0W > 0) + (K1W > 0); }
  __host__ __device__ static constexpr int kw(const Plan&, int i) { return i == 0 ? K0W : K1W; }
  __host__ __device__ static constexpr uint64_t kmask(const Plan&, int i) {
    return (i == 0 ? K0W : K1W) >= 8 ? ~0ULL : ((1ULL << (8 * (i == 0 ? K0W : K1W))) - 1);
  }
  __host__ __device__ static constexpr int kshift(const Plan&, int i) { return i == 0 ? 8 * K1W : 0; }
  __host__ __device__ static constexpr int nv(const Plan&) { return NVS; }
  __host__ __device__ static constexpr int kind(const Plan&, int v) { return (int)(op(v) & 3); }
  __host__ __device__ static constexpr int ia(int v) { return (int)((op(v) >> 2) & 7); }
  __host__ __device__ static constexpr int ib(int v) { return (int)((op(v) >> 5) & 7); }
  __host__ __device__ static constexpr int ic(int v) { return (int)((op(v) >> 8) & 7); }
  __host__ __device__ static constexpr bool fsum(const Plan&, int v) { return (op(v) >> 11) & VF_SUM; }
  __host__ __device__ static constexpr bool fmn(const Plan&, int v) { return (op(v) >> 11) & VF_MIN; }
  __host__ __device__ static constexpr bool fmx(const Plan&, int v) { return (op(v) >> 11) & VF_MAX; }
  __host__ __device__ static constexpr bool vf64(const Plan&, int) { return F64; }
  __device__ static bool special(Key k) {
    if constexpr (KBITS > 0 && KBITS < 32) return false;        // narrow keys can never be ~0
    else return k == (Key)~0ULL;
  }
  // Private-record layout at compile time; the planner (abi.cu plan_values) builds the
  // same layout at run time and shape_match checks they agree.  field: 0 sum, 1 hi, 2 min, 3 max.
  __host__ __device__ static constexpr int po_field(int v, int field) {
    int rec = 4, out = -1;
    for (int i = 0; i <= v; ++i) {
      const uint32_t f = op(i) >> 11;
      int ps = -1, ph = -1, pn = -1, px = -1;
      if (f & VF_SUM) {
        rec = (rec + 7) & ~7;
        ps = rec;
        rec += 8;
        if (!F64 && (op(i) & 3) != 0) { ph = rec; rec += 4; }
      }
      if (f & VF_MIN) { rec = (rec + 7) & ~7; pn = rec; rec += 8; }
      if (f & VF_MAX) { rec = (rec + 7) & ~7; px = rec; rec += 8; }
      if (i == v) out = field == 0 ? ps : field == 1 ? ph : field == 2 ? pn : px;
    }
    return out;
  }
  __host__ __device__ static constexpr int rec_bytes() {
    int rec = 4;
    for (int i = 0; i < NVS; ++i) {
      const uint32_t f = op(i) >> 11;
      if (f & VF_SUM) { rec = ((rec + 7) & ~7) + 8; if (!F64 && (op(i) & 3) != 0) rec += 4; }
      if (f & VF_MIN) rec = ((rec + 7) & ~7) + 8;
      if (f & VF_MAX) rec = ((rec + 7) & ~7) + 8;
    }
    return (rec + 7) & ~7;
  }
  __host__ __device__ static constexpr int po_sum(const Plan&, int v) { return po_field(v, 0); }
  __host__ __device__ static constexpr int po_hi(const Plan&, int v) { return po_field(v, 1); }
  __host__ __device__ static constexpr int po_min(const Plan&, int v) { return po_field(v, 2); }
  __host__ __device__ static constexpr int po_max(const Plan&, int v) { return po_field(v, 3); }
  __host__ __device__ static constexpr int rec(const Plan&) { return rec_bytes(); }
};

// ------------------------------------------------------------------ row evaluation
// Non-zero iff x does not fit int32: the high word differs from the sign of the low
// word (SHF + LOP3; checks are OR-ed and tested once per row).
__device__ __forceinline__ uint32_t i32_bad(int64_t x) {
  return (uint32_t)((uint64_t)x >> 32) ^ (uint32_t)((int32_t)(uint32_t)x >> 31);
}

template <class Sh, int NV, bool F64>
struct Row {
  bool q, fast;
  uint32_t bad;                            // int32 range violations of the fast path (0 = none)
  typename Sh::Key key;
  int64_t vi[F64 ? 1 : NV];
  double vd[F64 ? NV : 1];
};

template <int W>
__device__ __forceinline__ void ld2c(const void* base, int64_t r, uint64_t& x0, uint64_t& x1) {
  if constexpr (W == 1) {
    uint32_t v = __ldg((const unsigned short*)((const uint8_t*)base + r));
    x0 = v & 0xFF;
    x1 = v >> 8;
  } else if constexpr (W == 4) {
    int2 v = __ldg((const int2*)((const int32_t*)base + r));
    x0 = (uint64_t)(int64_t)v.x;
    x1 = (uint64_t)(int64_t)v.y;
  } else {
    longlong2 v = __ldg((const longlong2*)((const long long*)base + r));
    x0 = (uint64_t)v.x;
    x1 = (uint64_t)v.y;
  }
}

// 2-row load with a width that is a compile-time constant for static shapes.
__device__ __forceinline__ void ld2w(int w, const void* base, int64_t r, uint64_t& x0, uint64_t& x1) {
  if (w == 1) ld2c<1>(base, r, x0, x1);
  else if (w == 4) ld2c<4>(base, r, x0, x1);
  else ld2c<8>(base, r, x0, x1);
}
__device__ __forceinline__ uint64_t ld1w(int w, const void* base, int64_t r) {
  if (w == 1) return __ldg((const uint8_t*)base + r);
  if (w == 4) return (uint64_t)(int64_t)__ldg((const int32_t*)base + r);
  return (uint64_t)__ldg((const long long*)base + r);
}

__device__ __forceinline__ int64_t mul_wide_s32(int32_t a, int32_t b) {
  int64_t r;
  asm("mul.wide.s32 %0, %1, %2;" : "=l"(r) : "r"(a), "r"(b));
  return r;
}

template <class Sh>
__device__ __forceinline__ bool pred_ok(const Plan& p, int i, uint64_t raw) {
  const DevPred& d = p.preds[i];
  bool ok;
  if (Sh::pf64(p, i)) {
    const double x = __longlong_as_double((long long)raw);
    ok = x >= d.flo && x <= d.fhi;
  } else if (Sh::pw(p, i) < 8) {
    const int32_t x = (int32_t)(uint32_t)raw;                // u8 / i32: 32-bit compare on clamped bounds
    ok = x >= d.lo32 && x <= d.hi32;
  } else {
    const int64_t x = (int64_t)raw;
    ok = x >= d.lo && x <= d.hi;
  }
  return ok != (bool)d.anti;
}

// Value v of one row from its raw operands.  Integer fast path: COL values that fit
// int32 (accumulated in 64 bits), products of int32 factors via mul.wide.s32 (exact
// in int64); anything else clears `fast` (the row takes the exact int128 path).
template <class Sh, int NV, bool F64>
__device__ __forceinline__ void value_of(const Plan& p, int v, uint64_t ra, uint64_t rb, uint64_t rc,
                                         Row<Sh, NV, F64>& x) {
  const DevValue& d = p.vals[v];
  const int kind = Sh::kind(p, v);
  if constexpr (F64) {
    const double a = __longlong_as_double((long long)ra);
    if (kind == OCL_EXPR_COL) {
      x.vd[v] = a;
    } else {
      double e = __dmul_rn(a, __dsub_rn(d.Sf, __longlong_as_double((long long)rb)));
      if (kind == OCL_EXPR_MUL_1MINUS_1PLUS) e = __dmul_rn(e, __dadd_rn(d.Sf, __longlong_as_double((long long)rc)));
      x.vd[v] = e;
    }
  } else {
    const int64_t a = (int64_t)ra;
    if (kind == OCL_EXPR_COL) {
#if OCL_VAR_FITS
      x.fast = x.fast && fits_i32(a);
#else
      x.bad |= i32_bad(a);
#endif
      x.vi[v] = a;
    } else {
      const int64_t t = (int64_t)((uint64_t)d.S - rb);
#if OCL_VAR_FITS
      x.fast = x.fast && fits_i32(a) && fits_i32(t);
#else
      x.bad |= i32_bad(a) | i32_bad(t);
#endif
      int64_t e = mul_wide_s32((int32_t)a, (int32_t)t);
      if (kind == OCL_EXPR_MUL_1MINUS_1PLUS) {
        const int64_t u = (int64_t)((uint64_t)d.S + rc);
#if OCL_VAR_FITS
        x.fast = x.fast && fits_i32(e) && fits_i32(u);
#else
        x.bad |= i32_bad(e) | i32_bad(u);
#endif
        e = mul_wide_s32((int32_t)e, (int32_t)u);
      }
      x.vi[v] = e;
    }
  }
}

template <class Sh>
__device__ __forceinline__ typename Sh::Key pack_key(const Plan& p, const uint64_t* raw) {
  typename Sh::Key k = 0;
#pragma unroll
  for (int i = 0; i < kMaxKeys; ++i) {
    if (i >= Sh::nk(p)) break;
    k |= (typename Sh::Key)((raw[i] & Sh::kmask(p, i)) << Sh::kshift(p, i));
  }
  return k;
}

// Both rows of a lane's 64-row unit (vector loads; full tiles only).
template <class Sh, int NV, bool F64>
__device__ __forceinline__ void eval_pair(const Plan& p, int64_t r, Row<Sh, NV, F64>& x0, Row<Sh, NV, F64>& x1) {
  x0.q = x1.q = true;
  x0.fast = x1.fast = true;
  x0.bad = x1.bad = 0;
#pragma unroll
  for (int i = 0; i < kMaxPreds; ++i) {
    if (i >= Sh::np(p)) break;
    uint64_t u0, u1;
    ld2w(Sh::pw(p, i), p.preds[i].col.ptr, r, u0, u1);
    x0.q = x0.q && pred_ok<Sh>(p, i, u0);
    x1.q = x1.q && pred_ok<Sh>(p, i, u1);
  }
  uint64_t k0[kMaxKeys] = {0, 0}, k1[kMaxKeys] = {0, 0};
#pragma unroll
  for (int i = 0; i < kMaxKeys; ++i) {
    if (i >= Sh::nk(p)) break;
    ld2w(Sh::kw(p, i), p.keys[i].col.ptr, r, k0[i], k1[i]);
  }
  x0.key = pack_key<Sh>(p, k0);
  x1.key = pack_key<Sh>(p, k1);
  if constexpr (Sh::kStatic) {
    uint64_t c0[Sh::NC], c1[Sh::NC];      // every distinct value column loaded once
#pragma unroll
    for (int i = 0; i < Sh::NC; ++i) ld2c<8>(p.vcols[i].ptr, r, c0[i], c1[i]);
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      value_of<Sh, NV, F64>(p, v, c0[Sh::ia(v)], c0[Sh::ib(v)], c0[Sh::ic(v)], x0);
      value_of<Sh, NV, F64>(p, v, c1[Sh::ia(v)], c1[Sh::ib(v)], c1[Sh::ic(v)], x1);
    }
  } else {
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      if (v >= p.nvals) break;
      const DevValue& d = p.vals[v];
      if (!F64 && d.is_f64) {              // mixed int/fp64 plan: fp64 values take the exact slow path
        x0.fast = x1.fast = false;
        continue;
      }
      uint64_t a0, a1, b0 = 0, b1 = 0, c0 = 0, c1 = 0;
      ld2w(d.a.width, d.a.ptr, r, a0, a1);
      if (d.expr >= OCL_EXPR_MUL_1MINUS) ld2w(d.b.width, d.b.ptr, r, b0, b1);
      if (d.expr >= OCL_EXPR_MUL_1MINUS_1PLUS) ld2w(d.c.width, d.c.ptr, r, c0, c1);
      value_of<Sh, NV, F64>(p, v, a0, b0, c0, x0);
      value_of<Sh, NV, F64>(p, v, a1, b1, c1, x1);
    }
  }
  x0.fast = x0.fast && x0.bad == 0;
  x1.fast = x1.fast && x1.bad == 0;
}

// Static shapes: raw column words of one 64-row unit (both rows of the lane), loaded
// for every unit of a tile before any row is evaluated (loads in flight, few live
// registers: values are computed per unit just before they are placed).
template <class Sh>
struct RawUnit {
  uint64_t pr[2];
  uint64_t k[2][kMaxKeys];
  uint64_t c[2][Sh::NC];
};

template <class Sh>
__device__ __forceinline__ void load_unit(const Plan& p, int64_t r, RawUnit<Sh>& u) {
  if constexpr (Sh::kStatic) {
    if (Sh::np(p) > 0) ld2w(Sh::pw(p, 0), p.preds[0].col.ptr, r, u.pr[0], u.pr[1]);
#pragma unroll
    for (int i = 0; i < kMaxKeys; ++i) {
      if (i >= Sh::nk(p)) break;
      ld2w(Sh::kw(p, i), p.keys[i].col.ptr, r, u.k[0][i], u.k[1][i]);
    }
#pragma unroll
    for (int i = 0; i < Sh::NC; ++i) ld2c<8>(p.vcols[i].ptr, r, u.c[0][i], u.c[1][i]);
  }
}

template <class Sh, int NV, bool F64>
__device__ __forceinline__ void eval_unit(const Plan& p, const RawUnit<Sh>& u, int k, Row<Sh, NV, F64>& x) {
  if constexpr (Sh::kStatic) {
    x.q = Sh::np(p) > 0 ? pred_ok<Sh>(p, 0, u.pr[k]) : true;
    x.fast = true;
    x.bad = 0;
    uint64_t kk[kMaxKeys] = {0, 0};
#pragma unroll
    for (int i = 0; i < kMaxKeys; ++i) {
      if (i >= Sh::nk(p)) break;
      kk[i] = u.k[k][i];
    }
    x.key = pack_key<Sh>(p, kk);
#pragma unroll
    for (int v = 0; v < NV; ++v) value_of<Sh, NV, F64>(p, v, u.c[k][Sh::ia(v)], u.c[k][Sh::ib(v)], u.c[k][Sh::ic(v)], x);
    x.fast = x.fast && x.bad == 0;
  }
}

// One row with scalar loads (ragged tail, unaligned columns).
template <class Sh, int NV, bool F64>
__device__ __forceinline__ void eval_one(const Plan& p, int64_t r, Row<Sh, NV, F64>& x) {
  x.fast = true;
  x.bad = 0;
  x.key = 0;
  x.q = r < p.n;
  if (!x.q) return;
#pragma unroll
  for (int i = 0; i < kMaxPreds; ++i) {
    if (i >= Sh::np(p)) break;
    x.q = x.q && pred_ok<Sh>(p, i, ld1w(Sh::pw(p, i), p.preds[i].col.ptr, r));
  }
  uint64_t k[kMaxKeys] = {0, 0};
#pragma unroll
  for (int i = 0; i < kMaxKeys; ++i) {
    if (i >= Sh::nk(p)) break;
    k[i] = ld1w(Sh::kw(p, i), p.keys[i].col.ptr, r);
  }
  x.key = pack_key<Sh>(p, k);
#pragma unroll
  for (int v = 0; v < NV; ++v) {
    if (v >= Sh::nv(p)) break;
    const DevValue& d = p.vals[v];
    if (!F64 && d.is_f64) {
      x.fast = false;
      continue;
    }
    const uint64_t a = ld1w(d.a.width, d.a.ptr, r);
    const uint64_t b = d.expr >= OCL_EXPR_MUL_1MINUS ? ld1w(d.b.width, d.b.ptr, r) : 0;
    const uint64_t c = d.expr >= OCL_EXPR_MUL_1MINUS_1PLUS ? ld1w(d.c.width, d.c.ptr, r) : 0;
    value_of<Sh, NV, F64>(p, v, a, b, c, x);
  }
  x.fast = x.fast && x.bad == 0;
}

// ------------------------------------------------------------------ 1. private slots
// Record per thread per slot (offsets from the planner, Plan::priv_rec bytes):
// count u32; per value: SUM of a COL value as i64 (fast path: int32 values), SUM of a
// product as 96-bit (u64 lo + u32 hi), fp64 SUM as double; MIN / MAX as u64 order-
// preserving encodings (0 = identity).  Layout [slot][field][thread].
template <class Sh, int NV, bool F64>
__device__ __forceinline__ void priv_add(const Plan& p, uint8_t* sm, int slot, int tid, const Row<Sh, NV, F64>& x) {
  constexpr int T = kFusedThreads;
  uint8_t* base = sm + (size_t)slot * Sh::rec(p) * T;
  ((uint32_t*)base)[tid] += 1u;
#pragma unroll
  for (int v = 0; v < NV; ++v) {
    if (v >= Sh::nv(p)) break;
    if constexpr (F64) {
      const double val = x.vd[v];
      if (Sh::fsum(p, v)) ((double*)(base + Sh::po_sum(p, v) * T))[tid] += val;
      if (Sh::fmn(p, v)) {
        uint64_t* m = (uint64_t*)(base + Sh::po_min(p, v) * T) + tid;
        *m = max(*m, enc_min_f(val));
      }
      if (Sh::fmx(p, v)) {
        uint64_t* m = (uint64_t*)(base + Sh::po_max(p, v) * T) + tid;
        *m = max(*m, enc_max_f(val));
      }
    } else {
      if (Sh::vf64(p, v)) continue;
      const int64_t val = x.vi[v];
      if (Sh::fsum(p, v)) {
        if (Sh::kind(p, v) == OCL_EXPR_COL) {
          ((int64_t*)(base + Sh::po_sum(p, v) * T))[tid] += (int64_t)(int32_t)val;
        } else {
          uint64_t* lo = (uint64_t*)(base + Sh::po_sum(p, v) * T) + tid;
          uint32_t* hi = (uint32_t*)(base + Sh::po_hi(p, v) * T) + tid;
          uint64_t l = *lo;
          uint32_t h = *hi;
          uint32_t l0 = (uint32_t)l, l1 = (uint32_t)(l >> 32);
          asm("add.cc.u32 %0, %0, %3;\n\taddc.cc.u32 %1, %1, %4;\n\taddc.u32 %2, %2, %5;"
              : "+r"(l0), "+r"(l1), "+r"(h)
              : "r"((uint32_t)(uint64_t)val), "r"((uint32_t)((uint64_t)val >> 32)), "r"((uint32_t)(val >> 63)));
          *lo = (uint64_t)l0 | ((uint64_t)l1 << 32);
          *hi = h;
        }
      }
      if (Sh::fmn(p, v)) {
        uint64_t* m = (uint64_t*)(base + Sh::po_min(p, v) * T) + tid;
        *m = max(*m, enc_min_i(val));
      }
      if (Sh::fmx(p, v)) {
        uint64_t* m = (uint64_t*)(base + Sh::po_max(p, v) * T) + tid;
        *m = max(*m, enc_max_i(val));
      }
    }
  }
}

// ------------------------------------------------------------------ 2. CTA table
// [~key u64][count u32] per value: [sum of low 16 bits u32][sum of high 16 bits s32]
// [min u32][max u32] (order-preserving encodings, 0 = identity); int32 values only,
// 2^16 updates per field between flushes.  64-bit CAS on the key, linear probing.
constexpr int kSmemProbes = 16;
constexpr int kCtaFlushRounds = 64;   // 64 rounds x 8 warps x 128 rows = 65,536 rows

__device__ __forceinline__ uint8_t* cta_find_or_insert(uint8_t* tab, uint32_t cap, int32_t stride, uint64_t key) {
  const uint64_t sk = ~key;
  uint32_t h = (uint32_t)fmix64(key) & (cap - 1);
  for (int probe = 0; probe < kSmemProbes; ++probe) {
    uint64_t* kp = (uint64_t*)(tab + (size_t)h * stride);
    uint64_t cur = *(volatile uint64_t*)kp;
    if (cur == sk) return (uint8_t*)kp;
    if (cur == 0) {
      uint64_t prev = atomicCAS((unsigned long long*)kp, 0ULL, (unsigned long long)sk);
      if (prev == 0 || prev == sk) return (uint8_t*)kp;
    }
    h = (h + 1) & (cap - 1);
  }
  return nullptr;
}

__device__ __forceinline__ uint32_t enc32_max(int32_t v) { return (uint32_t)v ^ 0x80000000u; }
__device__ __forceinline__ uint32_t enc32_min(int32_t v) { return ~enc32_max(v); }

template <class Sh, int NV, bool F64>
__device__ __forceinline__ void cta_add(const Plan& p, uint8_t* e, const Row<Sh, NV, F64>& x) {
  atomicAdd((unsigned int*)(e + 8), 1u);
  if constexpr (!F64) {
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      if (v >= Sh::nv(p)) break;
      const DevValue& d = p.vals[v];
      const int32_t w = (int32_t)x.vi[v];
      if (Sh::fsum(p, v)) {
        atomicAdd((unsigned int*)(e + d.co_lo), (unsigned int)w & 0xFFFFu);
        atomicAdd((int*)(e + d.co_hi), w >> 16);
      }
      if (Sh::fmn(p, v)) atomicMax((unsigned int*)(e + d.co_min), enc32_min(w));
      if (Sh::fmx(p, v)) atomicMax((unsigned int*)(e + d.co_max), enc32_max(w));
    }
  }
}

// Fold one CTA-table entry into the HBM table and reset its accumulators (key kept).
// Direct mode (grouped aggregation over gids): the entry index is the group id.
__device__ __forceinline__ void cta_flush_entry(const Plan& p, uint8_t* ce, int64_t index = -1) {
  const uint64_t sk = *(const uint64_t*)ce;
  const uint32_t cnt = *(const uint32_t*)(ce + 8);
  if ((sk == 0 && index < 0) || cnt == 0) return;
  uint8_t* e = index >= 0 ? p.table + index * (int64_t)p.stride
                          : table_find_or_insert(p.table, p.mask, p.stride, ~sk, p.status);
  if (e) {
    atomicAdd((unsigned long long*)(e + 8), (unsigned long long)cnt);
    for (int v = 0; v < p.nvals; ++v) {
      const DevValue& d = p.vals[v];
      if (d.co_lo >= 0) {
        const int64_t sum =
            (int64_t)(*(const int32_t*)(ce + d.co_hi)) * 65536 + (int64_t)(*(const uint32_t*)(ce + d.co_lo));
        atomic_add_i128((uint64_t*)(e + d.off_sum), (uint64_t)sum, (uint64_t)(sum >> 63));
      }
      if (d.co_min >= 0) {
        const int32_t mn = (int32_t)(~*(const uint32_t*)(ce + d.co_min) ^ 0x80000000u);
        atomicMax((unsigned long long*)(e + d.off_min), (unsigned long long)enc_min_i(mn));
      }
      if (d.co_max >= 0) {
        const int32_t mx = (int32_t)(*(const uint32_t*)(ce + d.co_max) ^ 0x80000000u);
        atomicMax((unsigned long long*)(e + d.off_max), (unsigned long long)enc_max_i(mx));
      }
    }
  }
  for (int w = 8; w < p.cta_stride; w += 4) *(uint32_t*)(ce + w) = 0;
}

// ------------------------------------------------------------------ 3. HBM table (warp-aggregated)
// HBM entry of a key: hash table (fused path) or direct index (grouped aggregation
// over dense group ids, Plan::direct).
__device__ __forceinline__ uint8_t* resolve_entry(const Plan& p, uint64_t key) {
  if (p.direct) return p.table + key * (uint64_t)p.stride;
  return table_find_or_insert(p.table, p.mask, p.stride, key, p.status);
}

// Warp-reduce one private slot record (this warp's 32 lanes) and add it into entry e
// (a CTA-level entry in shared memory or an HBM entry).
__device__ __forceinline__ void priv_flush_warp(const Plan& p, const uint8_t* rec, int tid, uint8_t* e) {
  constexpr int T = kFusedThreads;
  const int lane = tid & 31;
  const uint32_t c = __reduce_add_sync(0xffffffffu, ((const uint32_t*)rec)[tid]);
  if (c == 0) return;                                 // warp-uniform
  if (lane == 0) atomicAdd((unsigned long long*)(e + 8), (unsigned long long)c);
  for (int v = 0; v < p.nvals; ++v) {
    const DevValue& d = p.vals[v];
    if (d.po_sum >= 0) {
      if (d.is_f64) {
        double sum = ((const double*)(rec + d.po_sum * T))[tid];
        for (int o = 16; o > 0; o >>= 1) sum += __shfl_xor_sync(0xffffffffu, sum, o);
        if (lane == 0) atomicAdd((double*)(e + d.off_sum), sum);
      } else {
        I128 x;
        x.lo = ((const uint64_t*)(rec + d.po_sum * T))[tid];
        x.hi = d.po_hi >= 0 ? (uint64_t)(int64_t)(int32_t)((const uint32_t*)(rec + d.po_hi * T))[tid]
                            : (uint64_t)((int64_t)x.lo >> 63);
        x = warp_sum_i128(x);
        if (lane == 0) atomic_add_i128((uint64_t*)(e + d.off_sum), x.lo, x.hi);
      }
    }
    if (d.po_min >= 0) {
      unsigned long long m = ((const uint64_t*)(rec + d.po_min * T))[tid];
      for (int o = 16; o > 0; o >>= 1) m = max(m, __shfl_xor_sync(0xffffffffu, m, o));
      if (lane == 0 && m) atomicMax((unsigned long long*)(e + d.off_min), m);
    }
    if (d.po_max >= 0) {
      unsigned long long m = ((const uint64_t*)(rec + d.po_max * T))[tid];
      for (int o = 16; o > 0; o >>= 1) m = max(m, __shfl_xor_sync(0xffffffffu, m, o));
      if (lane == 0 && m) atomicMax((unsigned long long*)(e + d.off_max), m);
    }
  }
}

// Add a whole entry (CTA-level, shared memory) into an HBM entry.
__device__ __forceinline__ void entry_merge(const Plan& p, const uint8_t* src, uint8_t* e) {
  atomicAdd((unsigned long long*)(e + 8), (unsigned long long)*(const uint64_t*)(src + 8));
  for (int v = 0; v < p.nvals; ++v) {
    const DevValue& d = p.vals[v];
    if (d.off_sum >= 0) {
      if (d.is_f64) atomicAdd((double*)(e + d.off_sum), *(const double*)(src + d.off_sum));
      else atomic_add_i128((uint64_t*)(e + d.off_sum), *(const uint64_t*)(src + d.off_sum),
                           *(const uint64_t*)(src + d.off_sum + 8));
    }
    if (d.off_min >= 0) atomicMax((unsigned long long*)(e + d.off_min), *(const unsigned long long*)(src + d.off_min));
    if (d.off_max >= 0) atomicMax((unsigned long long*)(e + d.off_max), *(const unsigned long long*)(src + d.off_max));
  }
}
template <int NV, bool F64>
struct MissStage {
  int64_t vi[F64 ? 1 : NV][32];
  double vd[F64 ? NV : 1][32];
};

template <class Sh, int NV, bool F64>
__device__ __forceinline__ void warp_miss_update(const Plan& p, MissStage<NV, F64>& st, bool miss,
                                                 const Row<Sh, NV, F64>& x, int lane) {
  const unsigned mmask = __ballot_sync(0xffffffffu, miss);
  if (mmask == 0) return;
  if (miss) {
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      if constexpr (F64) st.vd[v][lane] = x.vd[v];
      else st.vi[v][lane] = x.vi[v];
    }
  }
  __syncwarp();
  if (miss) {
    const unsigned peers = __match_any_sync(mmask, (unsigned long long)x.key);
    if (lane == __ffs(peers) - 1) {
      uint8_t* e = resolve_entry(p, (uint64_t)x.key);
      if (e) {
        atomicAdd((unsigned long long*)(e + 8), (unsigned long long)__popc(peers));
#pragma unroll
        for (int v = 0; v < NV; ++v) {
          if (v >= Sh::nv(p)) break;
          const DevValue& d = p.vals[v];
          if constexpr (F64) {
            double sum = 0.0, mn = x.vd[v], mx = x.vd[v];
            for (unsigned b = peers; b; b &= b - 1) {
              const double y = st.vd[v][__ffs(b) - 1];
              sum += y;
              mn = fmin(mn, y);
              mx = fmax(mx, y);
            }
            if (Sh::fsum(p, v)) atomicAdd((double*)(e + d.off_sum), sum);
            if (Sh::fmn(p, v)) atomicMax((unsigned long long*)(e + d.off_min), (unsigned long long)enc_min_f(mn));
            if (Sh::fmx(p, v)) atomicMax((unsigned long long*)(e + d.off_max), (unsigned long long)enc_max_f(mx));
          } else {
            if (Sh::vf64(p, v)) continue;
            I128 sum{0, 0};
            int64_t mn = x.vi[v], mx = x.vi[v];
            for (unsigned b = peers; b; b &= b - 1) {
              const int64_t y = st.vi[v][__ffs(b) - 1];
              sum = i128_add(sum, i128_from_i64(y));
              mn = min(mn, y);
              mx = max(mx, y);
            }
            if (Sh::fsum(p, v)) atomic_add_i128((uint64_t*)(e + d.off_sum), sum.lo, sum.hi);
            if (Sh::fmn(p, v)) atomicMax((unsigned long long*)(e + d.off_min), (unsigned long long)enc_min_i(mn));
            if (Sh::fmx(p, v)) atomicMax((unsigned long long*)(e + d.off_max), (unsigned long long)enc_max_i(mx));
          }
        }
      }
    }
  }
  __syncwarp();
}

// ------------------------------------------------------------------ per-row dispatch
template <class Sh, int NV, bool F64, bool MISS>
__device__ __forceinline__ void place_row(const Plan& p, uint64_t* dir, typename Sh::Key (&rk)[kRegSlots],
                                          uint8_t* sm, uint8_t* cta_tab, int tid, MissStage<MISS ? NV : 1, F64>& stage,
                                          const Row<Sh, NV, F64>& x, int64_t r) {
  using Key = typename Sh::Key;
  constexpr int L = kRegSlots;
  int slot = -1;
#pragma unroll
  for (int s = L - 1; s >= 0; --s)
    if (x.key == rk[s]) slot = s;
  const bool special = Sh::special(x.key);
  bool go = x.q && x.fast && slot >= 0 && !special;
  bool miss = false;
  if (x.q && !go) {                       // new key in this CTA, a slow value, or more keys than slots
    slot = (x.fast && !special) ? dir_find_or_insert<L>(dir, (uint64_t)x.key) : -1;
    if (slot >= 0) {
#pragma unroll
      for (int s = 0; s < L; ++s) {
        const uint64_t sk = *(volatile uint64_t*)&dir[s];
        rk[s] = sk ? (Key)~sk : (Key)~0ULL;
      }
      go = true;
    } else {
      uint8_t* e = nullptr;
      if constexpr (Sh::kCta) {
        if (p.smem_cap && x.fast && !special) e = cta_find_or_insert(cta_tab, (uint32_t)p.smem_cap, p.cta_stride, x.key);
      }
      if (e) {
        cta_add<Sh, NV, F64>(p, e, x);
      } else if (MISS && x.fast && !special) {
        miss = true;                      // warp-aggregated HBM update below
      } else {
        e = table_find_or_insert(p.table, p.mask, p.stride, (uint64_t)x.key, p.status);
        if (e) update_entry_slow(p, e, r);
      }
    }
  }
  if (go) priv_add<Sh, NV, F64>(p, sm, slot, tid, x);
  if constexpr (MISS) warp_miss_update<Sh, NV, F64>(p, stage, miss, x, tid & 31);
}

// ------------------------------------------------------------------ static-shape matching (host)
// The value part of a plan (distinct 8-byte value columns, expressions, accumulator
// flags, private-record layout) equals the compile-time shape Sh.
template <class Sh>
inline bool values_match(const Plan& g) {
  if (g.nvals != Sh::nv(g) || g.ncols != Sh::NC || g.priv_rec != Sh::rec(g)) return false;
  for (int i = 0; i < g.ncols; ++i)
    if (g.vcols[i].width != 8 || (g.vcols[i].dtype == OCL_F64) != Sh::vf64(g, 0)) return false;
  for (int v = 0; v < g.nvals; ++v) {
    const DevValue& d = g.vals[v];
    if (d.expr != Sh::kind(g, v) || (bool)d.is_f64 != Sh::vf64(g, v)) return false;
    if ((d.off_sum >= 0) != Sh::fsum(g, v) || (d.off_min >= 0) != Sh::fmn(g, v) ||
        (d.off_max >= 0) != Sh::fmx(g, v))
      return false;
    if (d.po_sum != Sh::po_sum(g, v) || d.po_hi != Sh::po_hi(g, v) || d.po_min != Sh::po_min(g, v) ||
        d.po_max != Sh::po_max(g, v))
      return false;
    if (d.ia != Sh::ia(v)) return false;
    if (d.expr >= OCL_EXPR_MUL_1MINUS && d.ib != Sh::ib(v)) return false;
    if (d.expr >= OCL_EXPR_MUL_1MINUS_1PLUS && d.ic != Sh::ic(v)) return false;
  }
  return true;
}

// GROUP BY an i64 key, COUNT/SUM/MIN/MAX of one i64 column (config C3), and the same
// behind an i32 range predicate (config C5).
using ShK64 = StaticShape<0, false, 8, 0, 1, false, vop(0, VF_SUM | VF_MIN | VF_MAX, 0)>;
using ShP32K64 = StaticShape<4, false, 8, 0, 1, false, vop(0, VF_SUM | VF_MIN | VF_MAX, 0)>;

// Whole plan (predicate / key widths + values) equals the compile-time shape Sh.
template <class Sh>
inline bool shape_match(const Plan& g) {
  if (g.npreds != Sh::np(g) || g.nkeys != Sh::nk(g)) return false;
  for (int i = 0; i < g.npreds; ++i)
    if (g.preds[i].col.width != Sh::pw(g, i) || (bool)g.preds[i].is_f64 != Sh::pf64(g, i)) return false;
  for (int i = 0; i < g.nkeys; ++i)
    if (g.keys[i].col.width != Sh::kw(g, i)) return false;
  return values_match<Sh>(g);
}

}  // namespace ocl
