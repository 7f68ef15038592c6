// common.cuh — device helpers and the launch "plans" shared by the kernels of
// libocelot_b200.so (sm_100a only).  Nothing here is shared with the oracle.
#pragma once

#ifndef __CUDACC_RTC__   // NVRTC (jit.cu) compiles the device headers without the runtime headers
#include <cuda_runtime.h>
#endif
#include <stdint.h>

#include "ocelot_b200.h"

#if defined(__CUDA_ARCH__) && (__CUDA_ARCH__ < 1000)
#error "libocelot_b200 targets sm_100a (B200) only"
#endif

namespace ocl {

constexpr int kMaxCols = 8;    // distinct input columns of one fused call
constexpr int kMaxPreds = 4;   // conjunction of range predicates
constexpr int kMaxKeys = 2;    // group-by columns (packed <= 64 bits)
constexpr int kMaxVals = 6;    // distinct value expressions
constexpr int kMaxAggs = 16;

// ------------------------------------------------------------------ hashing
// Table keys are stored complemented (stored = ~key) so that an all-zero
// (cudaMemset) table is empty; the one key whose complement is 0 (key == ~0)
// lives in a dedicated side entry at index `cap` (§8(c) s8: every 64-bit key is legal).
__host__ __device__ __forceinline__ uint64_t fmix64(uint64_t k) {   // murmur3 finaliser (s6)
  k ^= k >> 33;
  k *= 0xff51afd7ed558ccdULL;
  k ^= k >> 33;
  k *= 0xc4ceb9fe1a85ec53ULL;
  k ^= k >> 33;
  return k;
}

// ------------------------------------------------------------------ accumulator states
// Entry layout (AoS, `stride` bytes, 16-aligned): [0] stored key, [8] count,
// [16..] accumulator states at byte offsets chosen by the host planner:
//   SUM of ints -> 16 B two's-complement int128 {lo, hi}
//   SUM of f64  -> 8 B double
//   MIN / MAX   -> 8 B order-preserving unsigned encoding, updated with atomicMax,
//                  so that the zero-initialised state is the identity element.
enum AccKind : int32_t { ACC_SUM_I = 0, ACC_SUM_F = 1, ACC_MIN_I = 2, ACC_MAX_I = 3, ACC_MIN_F = 4, ACC_MAX_F = 5 };

__host__ __device__ __forceinline__ uint64_t enc_max_i(int64_t x) { return (uint64_t)x ^ 0x8000000000000000ULL; }
__host__ __device__ __forceinline__ uint64_t enc_min_i(int64_t x) { return ~enc_max_i(x); }
__host__ __device__ __forceinline__ int64_t dec_max_i(uint64_t e) { return (int64_t)(e ^ 0x8000000000000000ULL); }
__host__ __device__ __forceinline__ int64_t dec_min_i(uint64_t e) { return dec_max_i(~e); }
// doubles: flip all bits of negatives, the sign bit of non-negatives -> unsigned order
__device__ __forceinline__ uint64_t enc_max_f(double d) {
  uint64_t b = (uint64_t)__double_as_longlong(d);
  return (b >> 63) ? ~b : (b | 0x8000000000000000ULL);
}
__device__ __forceinline__ uint64_t enc_min_f(double d) { return ~enc_max_f(d); }
__device__ __forceinline__ double dec_max_f(uint64_t e) {
  uint64_t b = (e >> 63) ? (e & 0x7FFFFFFFFFFFFFFFULL) : ~e;
  return __longlong_as_double((long long)b);
}
__device__ __forceinline__ double dec_min_f(uint64_t e) { return dec_max_f(~e); }

// Exact int128 accumulate into {lo, hi} with two 64-bit atomics (global or shared
// generic address): the carry out of the low word is detected from the value the
// atomic returns, so concurrent adds stay exact modulo 2^128.
__device__ __forceinline__ void atomic_add_i128(uint64_t* p, uint64_t lo, uint64_t hi) {
  unsigned long long old = atomicAdd((unsigned long long*)p, (unsigned long long)lo);
  uint64_t carry = (old + lo) < old ? 1ULL : 0ULL;
  uint64_t h = hi + carry;
  if (h) atomicAdd((unsigned long long*)(p + 1), (unsigned long long)h);
}

// int128 helpers on {lo, hi} register pairs
struct I128 {
  uint64_t lo, hi;
};
__device__ __forceinline__ I128 i128_from_i64(int64_t v) { return I128{(uint64_t)v, (uint64_t)(v >> 63)}; }
__device__ __forceinline__ I128 i128_add(I128 a, I128 b) {
  I128 r;
  r.lo = a.lo + b.lo;
  r.hi = a.hi + b.hi + (r.lo < a.lo ? 1ULL : 0ULL);
  return r;
}
// (a * b) mod 2^128 for a 128-bit a and 128-bit b
__device__ __forceinline__ I128 i128_mul(I128 a, I128 b) {
  I128 r;
  r.lo = a.lo * b.lo;
  r.hi = __umul64hi(a.lo, b.lo) + a.lo * b.hi + a.hi * b.lo;
  return r;
}

// Correctly rounded int128 -> double (s13): exact via the 64-bit path when the
// value fits, else round a 64-bit window with a sticky bit once.
__device__ __forceinline__ double i128_to_double(uint64_t lo, uint64_t hi) {
  bool neg = (int64_t)hi < 0;
  if ((hi == 0 && (int64_t)lo >= 0) || (hi == ~0ULL && (int64_t)lo < 0)) return __ll2double_rn((long long)lo);
  if (neg) {   // magnitude (two's complement negate)
    lo = ~lo + 1;
    hi = ~hi + (lo == 0 ? 1 : 0);
  }
  // magnitude >= 2^63 here; normalise so bit 127 is set
  int lz = hi ? __clzll((long long)hi) : 64 + __clzll((long long)lo);
  uint64_t nhi, nlo;
  if (lz == 0) { nhi = hi; nlo = lo; }
  else if (lz < 64) { nhi = (hi << lz) | (lo >> (64 - lz)); nlo = lo << lz; }
  else { nhi = lo << (lz - 64); nlo = 0; }
  uint64_t top = nhi | (nlo ? 1ULL : 0ULL);   // sticky: 64 bits > 53 + 2, one rounding is exact
  double d = __ull2double_rn(top);
  d = ldexp(d, 64 - lz);
  return neg ? -d : d;
}

// ------------------------------------------------------------------ launch plans
struct DevCol {
  const void* ptr;
  int32_t dtype;   // ocl_dtype
  int32_t width;   // bytes per element
};

struct DevPred {
  DevCol col;
  int32_t is_f64;
  int32_t anti;
  int64_t lo, hi;     // normalised inclusive integer bounds (lo > hi: empty range)
  int32_t lo32, hi32; // the same clamped to int32 (u8 / i32 columns compare in 32 bits)
  double flo, fhi;    // normalised inclusive fp64 bounds
};

struct DevKey {
  DevCol col;
  int32_t shift;      // packed key |= (raw & mask) << shift
  int32_t pad;
  uint64_t mask;
};

struct DevValue {
  DevCol a, b, c;                     // operand columns (b, c unused for EXPR_COL)
  int32_t expr;
  int32_t is_f64;
  int32_t off_sum, off_min, off_max;  // entry byte offsets, -1 if that state is not needed
  int32_t po_sum, po_hi, po_min, po_max;  // private-accumulator field offsets (bytes per thread), -1 if absent
  int32_t co_lo, co_hi, co_min, co_max;   // CTA-table 32-bit field offsets (bytes in the entry), -1 if absent
  int32_t ia, ib, ic;                 // operand indices into Plan::vcols (static shapes)
  int64_t S;                          // 10^scale
  double Sf;
};

// Everything one fused / aggregate launch needs (passed by value, __grid_constant__).
struct Plan {
  int64_t n;
  int32_t npreds, nkeys, nvals;
  int32_t vec_ok;       // every column pointer aligned for 2-row vector loads
  DevPred preds[kMaxPreds];
  DevKey keys[kMaxKeys];
  DevValue vals[kMaxVals];
  int32_t ncols;        // distinct value columns (operands of all value expressions)
  int32_t pad2_;
  DevCol vcols[kMaxCols];
  uint8_t* table;       // cap + 1 entries (side entry last)
  uint64_t mask;        // cap - 1 (cap is a power of two)
  int32_t stride;       // entry bytes
  int32_t has_minmax;
  int32_t priv_rec;     // private accumulator record: bytes per thread per group slot
  int32_t smem_cap;     // register tier: per-CTA shared-memory hash table entries (0 = none; power of two)
  int32_t cta_stride;   // bytes per CTA-table entry
  int32_t direct;       // 1: HBM table indexed by the key itself (grouped aggregation over dense gids)
  int32_t miss_agg;     // 1: rows that miss the private slots / CTA table are warp-aggregated (many groups)
  int32_t* status;      // device status word (may be null)
  uint32_t* bitmap_out; // optional selection bitmap
  const int32_t* gids;  // unfused aggregate: direct group ids (table indexed by gid)
  const uint32_t* oids; // unfused aggregate: row ids (null: identity)
  const int64_t* m_dev; // unfused aggregate: device row count (null: n)
  int64_t expected;     // the caller's expected_groups (picks the accumulation tier of the bulk kernels)
};

struct OutAgg {
  int32_t op;       // ocl_agg_op
  int32_t kind;     // AccKind of the state read (COUNT: -1)
  int32_t off;      // state byte offset
  int32_t is_f64;   // input column class
  void* out;
};

struct StateDesc {
  int32_t kind;     // AccKind
  int32_t off;      // entry byte offset
};

struct FinPlan {
  int32_t naggs;
  int32_t order_by_key;
  OutAgg aggs[kMaxAggs];
  int32_t nstates;  // distinct accumulator states (merge schema)
  int32_t stride;   // entry bytes
  StateDesc states[3 * kMaxVals];
  int64_t* keys_out;      // may be null (unfused aggregate)
  int64_t* ngroups_out;
  int64_t out_capacity;
  int32_t* status;
};

constexpr uint64_t kProbeWindow = 2048;   // HBM-table probe window (= partition.cu kPartCap)

__device__ __forceinline__ void set_status(int32_t* status, int32_t code) {
  if (status) atomicCAS(status, 0, code);
}

__device__ __forceinline__ uint64_t ld_relaxed_u64(const uint64_t* p) {
  uint64_t v;
  asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p));
  return v;
}

// Find-or-insert a key in the open-addressing table (linear probing, atomicCAS;
// P:L511-533 §4.1.4 adapted to a single pessimistic round).  Returns
// the entry, or nullptr (and sets OCL_ERR_CAPACITY) when the table is full.
__device__ __forceinline__ uint8_t* table_find_or_insert(uint8_t* table, uint64_t mask, int32_t stride,
                                                          uint64_t key, int32_t* status) {
  if (key == ~0ULL) {   // side entry: stored key field doubles as an occupancy flag
    uint8_t* e = table + (mask + 1) * (uint64_t)stride;
    if (ld_relaxed_u64((const uint64_t*)e) == 0) atomicExch((unsigned long long*)e, 1ULL);
    return e;
  }
  uint64_t sk = ~key;
  // start slot = the top log2(cap) bits of the hash: the keys of hash partition q
  // (top bits = q, partition.cu) occupy one contiguous slot range.  Probing wraps
  // inside the aligned window of kProbeWindow slots holding the start slot, so a
  // probe sequence never leaves its partition's range (partition.cu stores whole
  // ranges position by position); at load <= 1/2 a window overflows with
  // negligible probability, and the capacity status triggers the restart.
  const uint64_t W = mask < kProbeWindow - 1 ? mask : (uint64_t)(kProbeWindow - 1);
  uint64_t h = __umul64hi(fmix64(key), mask + 1);
  for (uint64_t probe = 0; probe <= W; ++probe) {
    uint64_t* kp = (uint64_t*)(table + h * (uint64_t)stride);
    uint64_t cur = ld_relaxed_u64(kp);
    if (cur == sk) return (uint8_t*)kp;
    if (cur == 0) {
      uint64_t prev = atomicCAS((unsigned long long*)kp, 0ULL, (unsigned long long)sk);
      if (prev == 0 || prev == sk) return (uint8_t*)kp;
    }
    h = (h & ~W) | ((h + 1) & W);
  }
  set_status(status, OCL_ERR_CAPACITY);
  return nullptr;
}

__host__ __device__ __forceinline__ int dtype_width(int32_t dt) {
  return dt == OCL_U8 ? 1 : (dt == OCL_I32 ? 4 : 8);
}

// Raw element (u8 zero-extended, i32 sign-extended, i64 / f64 bits) of a column.
__device__ __forceinline__ uint64_t load_raw(const DevCol& c, int64_t r) {
  switch (c.dtype) {
    case OCL_U8: return (uint64_t)__ldg((const uint8_t*)c.ptr + r);
    case OCL_I32: return (uint64_t)(int64_t)__ldg((const int32_t*)c.ptr + r);
    default: return (uint64_t)__ldg((const unsigned long long*)c.ptr + r);
  }
}

}  // namespace ocl
