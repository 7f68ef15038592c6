// rowops.cuh — per-row device operations of the fused path: predicate, key
// packing, value expressions, global-table update.  Used by fused.cu and
// aggregate.cu (product side only; independent of the oracle).
#pragma once

#include "common.cuh"

namespace ocl {

// Two consecutive elements of a column starting at an even row r, one vector load
// (u8: 2 B, i32: 8 B, i64/f64: 16 B).  Requires the column pointer aligned to
// 2 * width (checked on the host -> Plan::vec_ok).  Raw form: u8 zero-extended,
// i32 sign-extended, i64/f64 bits.
__device__ __forceinline__ void load_pair(const DevCol& c, int64_t r, uint64_t& x0, uint64_t& x1) {
  if (c.width == 1) {
    uint32_t v = __ldg((const unsigned short*)((const uint8_t*)c.ptr + r));
    x0 = v & 0xFF;
    x1 = v >> 8;
  } else if (c.width == 4) {
    int2 v = __ldg((const int2*)((const int32_t*)c.ptr + r));
    x0 = (uint64_t)(int64_t)v.x;
    x1 = (uint64_t)(int64_t)v.y;
  } else {
    longlong2 v = __ldg((const longlong2*)((const long long*)c.ptr + r));
    x0 = (uint64_t)v.x;
    x1 = (uint64_t)v.y;
  }
}

__device__ __forceinline__ uint64_t load_one(const DevCol& c, int64_t r) {
  if (c.width == 1) return (uint64_t)__ldg((const uint8_t*)c.ptr + r);
  if (c.width == 4) return (uint64_t)(int64_t)__ldg((const int32_t*)c.ptr + r);
  return (uint64_t)__ldg((const long long*)c.ptr + r);
}

// MonetDB range predicate on normalised inclusive bounds (s2); raw from load_*.
__device__ __forceinline__ bool eval_pred(const DevPred& p, uint64_t raw) {
  bool ok;
  if (p.is_f64) {
    double d = __longlong_as_double((long long)raw);
    ok = d >= p.flo && d <= p.fhi;
  } else {
    int64_t x = (int64_t)raw;
    ok = x >= p.lo && x <= p.hi;
  }
  return ok != (bool)p.anti;
}

// x fits int32 <=> its high word is the sign extension of its low word (2 SASS ops)
__device__ __forceinline__ bool fits_i32(int64_t x) {
  return (uint32_t)((uint64_t)x >> 32) == (uint32_t)((int32_t)(uint32_t)x >> 31);
}

// Integer value expression, fast path: exact in int64 when every factor fits in
// int32 (true for all TPC-H-ranged decimals); otherwise *fast = false and the row
// is re-evaluated in int128 by the slow path (value_i128).
__device__ __forceinline__ int64_t value_i64_fast(const DevValue& v, uint64_t ra, uint64_t rb, uint64_t rc, bool& fast) {
  int64_t a = (int64_t)ra;
  if (v.expr == OCL_EXPR_COL) return a;
  int64_t t = (int64_t)((uint64_t)v.S - rb);                 // S - b (wraps only when not int32-sized)
  fast = fast && fits_i32(a) && fits_i32(t);
  int64_t p = (int64_t)(int32_t)a * (int64_t)(int32_t)t;   // IMAD.WIDE: exact
  if (v.expr == OCL_EXPR_MUL_1MINUS) return p;
  int64_t u = (int64_t)((uint64_t)v.S + rc);
  fast = fast && fits_i32(p) && fits_i32(u);
  return (int64_t)(int32_t)p * (int64_t)(int32_t)u;
}

// Integer value expression in int128 modulo 2^128 (the ABI definition).
__device__ __forceinline__ I128 value_i128(const DevValue& v, uint64_t ra, uint64_t rb, uint64_t rc) {
  I128 a = i128_from_i64((int64_t)ra);
  if (v.expr == OCL_EXPR_COL) return a;
  I128 S = i128_from_i64(v.S);
  I128 nb = i128_from_i64((int64_t)rb);
  I128 t;                                   // S - b
  t.lo = S.lo - nb.lo;
  t.hi = S.hi - nb.hi - (S.lo < nb.lo ? 1ULL : 0ULL);
  I128 e = i128_mul(a, t);
  if (v.expr == OCL_EXPR_MUL_1MINUS) return e;
  I128 u = i128_add(S, i128_from_i64((int64_t)rc));
  return i128_mul(e, u);
}

// fp64 value expression: (a * (S - b)) * (S + c), left to right, no FMA (s14).
__device__ __forceinline__ double value_f64(const DevValue& v, uint64_t ra, uint64_t rb, uint64_t rc) {
  double a = __longlong_as_double((long long)ra);
  if (v.expr == OCL_EXPR_COL) return a;
  double e = __dmul_rn(a, __dsub_rn(v.Sf, __longlong_as_double((long long)rb)));
  if (v.expr == OCL_EXPR_MUL_1MINUS) return e;
  return __dmul_rn(e, __dadd_rn(v.Sf, __longlong_as_double((long long)rc)));
}

// Packed group key of row r (s5): raw bits masked to the column width.
__device__ __forceinline__ uint64_t row_key_scalar(const Plan& p, int64_t r) {
  uint64_t k = 0;
#pragma unroll
  for (int i = 0; i < kMaxKeys; ++i)
    if (i < p.nkeys) k |= (load_one(p.keys[i].col, r) & p.keys[i].mask) << p.keys[i].shift;
  return k;
}

__device__ __forceinline__ bool row_pred_scalar(const Plan& p, int64_t r) {
  bool q = true;
#pragma unroll
  for (int i = 0; i < kMaxPreds; ++i)
    if (i < p.npreds) q = q && eval_pred(p.preds[i], load_one(p.preds[i].col, r));
  return q;
}

// Apply the full contribution of row r (group entry e) with global atomics,
// re-reading its operands: the path for rows that miss the register tier or
// whose values need int128 (rare on the low-G path; every row on the global tier
// when called with precomputed values is handled by update_entry_fast below).
__device__ __forceinline__ void update_entry_slow(const Plan& p, uint8_t* e, int64_t r) {
  atomicAdd((unsigned long long*)(e + 8), 1ULL);
#pragma unroll
  for (int i = 0; i < kMaxVals; ++i) {
    if (i >= p.nvals) break;
    const DevValue& v = p.vals[i];
    uint64_t ra = load_one(v.a, r);
    uint64_t rb = v.expr >= OCL_EXPR_MUL_1MINUS ? load_one(v.b, r) : 0;
    uint64_t rc = v.expr >= OCL_EXPR_MUL_1MINUS_1PLUS ? load_one(v.c, r) : 0;
    if (v.is_f64) {
      double d = value_f64(v, ra, rb, rc);
      if (v.off_sum >= 0) atomicAdd((double*)(e + v.off_sum), d);
      if (v.off_min >= 0) atomicMax((unsigned long long*)(e + v.off_min), (unsigned long long)enc_min_f(d));
      if (v.off_max >= 0) atomicMax((unsigned long long*)(e + v.off_max), (unsigned long long)enc_max_f(d));
    } else {
      I128 x = value_i128(v, ra, rb, rc);
      if (v.off_sum >= 0) atomic_add_i128((uint64_t*)(e + v.off_sum), x.lo, x.hi);
      if (v.off_min >= 0) atomicMax((unsigned long long*)(e + v.off_min), (unsigned long long)enc_min_i((int64_t)x.lo));
      if (v.off_max >= 0) atomicMax((unsigned long long*)(e + v.off_max), (unsigned long long)enc_max_i((int64_t)x.lo));
    }
  }
}


__device__ __forceinline__ I128 warp_sum_i128(I128 x) {
#pragma unroll
  for (int o = 16; o > 0; o >>= 1) {
    I128 y;
    y.lo = __shfl_xor_sync(0xffffffffu, x.lo, o);
    y.hi = __shfl_xor_sync(0xffffffffu, x.hi, o);
    x = i128_add(x, y);
  }
  return x;
}

// Block-wide slot directory: stored keys (~key), 0 = free.  Returns slot or -1.
template <int L>
__device__ __forceinline__ int dir_find_or_insert(uint64_t* dir, uint64_t key) {
  uint64_t sk = ~key;
#pragma unroll
  for (int s = 0; s < L; ++s) {
    uint64_t cur = *(volatile uint64_t*)&dir[s];
    if (cur == sk) return s;
    if (cur == 0) {
      uint64_t prev = atomicCAS((unsigned long long*)&dir[s], 0ULL, (unsigned long long)sk);
      if (prev == 0 || prev == sk) return s;
    }
  }
  return -1;
}

// Optional bitmap output for a 64-row unit: rows base + 2*lane + {0,1}.
__device__ __forceinline__ void emit_bitmap_unit(const Plan& p, int64_t base, int lane, bool q0, bool q1) {
  uint32_t b = (uint32_t)q0 | ((uint32_t)q1 << 1);
  uint32_t w0 = __reduce_or_sync(0xffffffffu, lane < 16 ? b << (2 * lane) : 0u);
  uint32_t w1 = __reduce_or_sync(0xffffffffu, lane >= 16 ? b << (2 * (lane - 16)) : 0u);
  int64_t words = (p.n + 31) >> 5;
  int64_t wi = base >> 5;
  if (lane == 0 && wi < words) p.bitmap_out[wi] = w0;
  if (lane == 1 && wi + 1 < words) p.bitmap_out[wi + 1] = w1;
}

// Finalisation (§4.1.7: one thread per group computes the final aggregate).
// Decode one entry into output row g (finalize).
__device__ __forceinline__ void emit_final(const FinPlan& f, const uint8_t* e, uint64_t key, int64_t g) {
  if (g >= f.out_capacity) return;
  if (f.keys_out) f.keys_out[g] = (int64_t)key;
  const uint64_t count = *(const uint64_t*)(e + 8);
  for (int i = 0; i < f.naggs; ++i) {
    const OutAgg& a = f.aggs[i];
    const uint8_t* s = e + a.off;
    switch (a.op) {
      case OCL_AGG_COUNT: ((int64_t*)a.out)[g] = (int64_t)count; break;
      case OCL_AGG_SUM:
        if (a.is_f64) ((double*)a.out)[g] = *(const double*)s;
        else {
          ((uint64_t*)a.out)[2 * g] = *(const uint64_t*)s;
          ((uint64_t*)a.out)[2 * g + 1] = *(const uint64_t*)(s + 8);
        }
        break;
      case OCL_AGG_AVG: {
        double sum = a.is_f64 ? *(const double*)s : i128_to_double(*(const uint64_t*)s, *(const uint64_t*)(s + 8));
        ((double*)a.out)[g] = __ddiv_rn(sum, __ull2double_rn(count));
        break;
      }
      case OCL_AGG_MIN:
        if (a.is_f64) ((double*)a.out)[g] = dec_min_f(*(const uint64_t*)s);
        else ((int64_t*)a.out)[g] = dec_min_i(*(const uint64_t*)s);
        break;
      case OCL_AGG_MAX:
        if (a.is_f64) ((double*)a.out)[g] = dec_max_f(*(const uint64_t*)s);
        else ((int64_t*)a.out)[g] = dec_max_i(*(const uint64_t*)s);
        break;
    }
  }
}

}  // namespace ocl
