// spec_device.cuh — device code of the plan-signature fused kernels (k_sga_bulk, k_sga_priv):
// signatures, row evaluation, accumulation tiers, the TMA bulk pipeline.  Compiled twice:
// ahead of time by nvcc for the signatures fused_spec.cu instantiates, and at run time by
// NVRTC (jit.cu) for any other plan that fits a signature — Ocelot compiled its OpenCL
// kernels at run time for the device it ran on.  Design
// notes: fused_spec.cu and DESIGN.md §6.1.  No host-only code and no standard headers
// here (NVRTC gets this file, bulk.cuh, rowops.cuh, common.cuh, ocelot_b200.h).
#pragma once

#include "bulk.cuh"
#include "rowops.cuh"

namespace ocl {

template <bool C, class A, class B>
struct cond_t {
  using type = A;
};
template <class A, class B>
struct cond_t<false, A, B> {
  using type = B;
};

enum : uint32_t { VX_COL = 0, VX_M1 = 1, VX_M1P = 2 };
enum : uint32_t { VS_SUM = 1, VS_MIN = 2, VS_MAX = 4 };
// value descriptor: kind (2 bits) | a (3) | b (3) | c (3) | flags (3: SUM / MIN / MAX)
__host__ __device__ constexpr uint32_t vop(uint32_t kind, uint32_t a, uint32_t b = 0, uint32_t c = 0,
                                           uint32_t flags = VS_SUM) {
  return kind | (a << 2) | (b << 5) | (c << 8) | (flags << 11);
}
__host__ __device__ constexpr uint32_t vx_kind(uint32_t o) { return o & 3; }
__host__ __device__ constexpr uint32_t vx_a(uint32_t o) { return (o >> 2) & 7; }
__host__ __device__ constexpr uint32_t vx_b(uint32_t o) { return (o >> 5) & 7; }
__host__ __device__ constexpr uint32_t vx_c(uint32_t o) { return (o >> 8) & 7; }
__host__ __device__ constexpr uint32_t vx_flags(uint32_t o) { return (o >> 11) & 7; }

// PW: predicate column width (0 = no predicate); K0W/K1W: key widths (0 = absent);
// NC: distinct value columns (all i64, or all f64 when F64); OPS: value expressions.
template <int PW_, bool PF64_, int K0W_, int K1W_, int NC_, bool F64_, uint32_t... OPS>
struct Sig {
  static constexpr int PW = PW_;
  static constexpr bool PF64 = PF64_;
  static constexpr int K0W = K0W_, K1W = K1W_;
  static constexpr int NC = NC_;
  static constexpr bool F64 = F64_;
  static constexpr int NV = sizeof...(OPS);
  __host__ __device__ static constexpr uint32_t OP(int v) {
    const uint32_t a[NV] = {OPS...};
    return a[v];
  }
  static constexpr int KBITS = 8 * (K0W + K1W);
  static constexpr bool NARROW_KEY = KBITS < 32;   // 0xFFFFFFFF can never be a key
  __host__ __device__ static constexpr bool has(int v, uint32_t f) { return (vx_flags(OP(v)) & f) != 0; }
  // the CTA-table tier holds integer COL values (int32 fast path) only
  __host__ __device__ static constexpr bool cta_ok() {
    for (int v = 0; v < NV; ++v)
      if (vx_kind(OP(v)) != VX_COL) return false;
    return !F64;
  }
};

struct SpecPlan {
  Plan g;                     // generic plan (slow path, tail rows, flush offsets)
  const void* pcol;
  int32_t plo, phi;           // predicate bounds clamped to int32 (int columns)
  const void* k0;
  const void* k1;
  const void* col[4];
  uint32_t tab_hb;            // CTA-table tier: log2 of the slots per table (H)
  uint32_t tab_nrep;          // CTA-table tier: tables per CTA (1 by default)
  int32_t pwait, cwait;       // barrier wait strategies of the producer / consumers (mbar_wait_mode)
  int32_t mm_check;           // CTA-table tier: MIN / MAX atomics only when the value improves
  int32_t sparse_pct;         // select-compact-gather below this sampled selectivity (%); 0 = off
};

template <class S>
__device__ __forceinline__ bool spec_pred(const SpecPlan& p, uint64_t raw) {
  if constexpr (S::PW == 0) {
    return true;
  } else if constexpr (S::PF64) {
    double d = __longlong_as_double((long long)raw);
    return (d >= p.g.preds[0].flo && d <= p.g.preds[0].fhi) != (bool)p.g.preds[0].anti;
  } else if constexpr (S::PW == 8) {
    int64_t x = (int64_t)raw;
    return (x >= p.g.preds[0].lo && x <= p.g.preds[0].hi) != (bool)p.g.preds[0].anti;
  } else {
    int32_t x = (int32_t)(uint32_t)raw;
    return (x >= p.plo && x <= p.phi) != (bool)p.g.preds[0].anti;
  }
}

// 2-row vector load of a column of width W at even row r (raw u64 per row).
template <int W>
__device__ __forceinline__ void ld2(const void* base, int64_t r, uint64_t& x0, uint64_t& x1) {
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

template <int W>
__device__ __forceinline__ uint64_t ld1(const void* base, int64_t r) {
  if constexpr (W == 1) return __ldg((const uint8_t*)base + r);
  else if constexpr (W == 4) return (uint64_t)(int64_t)__ldg((const int32_t*)base + r);
  else return (uint64_t)__ldg((const long long*)base + r);
}

__device__ __forceinline__ int64_t spec_mul_wide_s32(int32_t a, int32_t b) {
  int64_t r;
  asm("mul.wide.s32 %0, %1, %2;" : "=l"(r) : "r"(a), "r"(b));
  return r;
}

// Non-zero iff x does not fit int32 (high word != sign of the low word).
__device__ __forceinline__ uint32_t spec_i32_bad(int64_t x) {
  return (uint32_t)((uint64_t)x >> 32) ^ (uint32_t)((int32_t)(uint32_t)x >> 31);
}

// order-preserving 32-bit encodings of int32 (zero-initialised = identity for a max)
__device__ __forceinline__ uint32_t s_enc32_max(int32_t v) { return (uint32_t)v ^ 0x80000000u; }
__device__ __forceinline__ uint32_t s_enc32_min(int32_t v) { return ~s_enc32_max(v); }
__device__ __forceinline__ int32_t s_dec32_max(uint32_t e) { return (int32_t)(e ^ 0x80000000u); }
__device__ __forceinline__ int32_t s_dec32_min(uint32_t e) { return s_dec32_max(~e); }

template <class S>
using KeyT = typename cond_t<(S::KBITS <= 32), uint32_t, uint64_t>::type;

template <class S>
__device__ __forceinline__ KeyT<S> spec_key(uint64_t k0, uint64_t k1) {
  if constexpr (S::K0W == 0) return 0;
  else if constexpr (S::K1W == 0) return (KeyT<S>)k0;
  else {
    constexpr uint64_t m0 = S::K0W == 8 ? ~0ULL : ((1ULL << (8 * S::K0W)) - 1);
    constexpr uint64_t m1 = S::K1W == 8 ? ~0ULL : ((1ULL << (8 * S::K1W)) - 1);
    return (KeyT<S>)(((k0 & m0) << (8 * S::K1W)) | (k1 & m1));
  }
}

// One row after evaluation: predicate, key, values on the fast path.
template <class S>
struct SRow {
  bool q, fast;
  KeyT<S> key;
  int64_t vi[S::F64 ? 1 : S::NV];
  double vd[S::F64 ? S::NV : 1];
};

// Values from the row's NC operand columns (compile-time expression program).
template <class S>
__device__ __forceinline__ void spec_values(const SpecPlan& p, const uint64_t (&c)[S::NC], SRow<S>& x) {
  uint32_t bad = 0;
#pragma unroll
  for (int v = 0; v < S::NV; ++v) {
    const uint32_t op = S::OP(v);
    const uint32_t kind = vx_kind(op);
    if constexpr (S::F64) {
      double a = __longlong_as_double((long long)c[vx_a(op)]);
      if (kind == VX_COL) {
        x.vd[v] = a;
      } else {
        double e = __dmul_rn(a, __dsub_rn(p.g.vals[v].Sf, __longlong_as_double((long long)c[vx_b(op)])));
        if (kind == VX_M1P) e = __dmul_rn(e, __dadd_rn(p.g.vals[v].Sf, __longlong_as_double((long long)c[vx_c(op)])));
        x.vd[v] = e;
      }
    } else {
      // int32 range checks OR-ed into one word (SHF + LOP3 each), tested once per row:
      // compare chains on 64-bit values cost ~5x more issue slots.
      int64_t a = (int64_t)c[vx_a(op)];
      if (kind == VX_COL) {
        bad |= spec_i32_bad(a);                          // narrow accumulator (64-bit) on the fast path
        x.vi[v] = a;
      } else {
        int64_t t = (int64_t)((uint64_t)p.g.vals[v].S - c[vx_b(op)]);
        bad |= spec_i32_bad(a) | spec_i32_bad(t);
        int64_t e = spec_mul_wide_s32((int32_t)a, (int32_t)t);
        if (kind == VX_M1P) {
          int64_t u = (int64_t)((uint64_t)p.g.vals[v].S + c[vx_c(op)]);
          bad |= spec_i32_bad(e) | spec_i32_bad(u);
          e = spec_mul_wide_s32((int32_t)e, (int32_t)u);
        }
        x.vi[v] = e;
      }
    }
  }
  if constexpr (!S::F64) x.fast = x.fast && bad == 0;
}

// ------------------------------------------------------------------ private accumulators
// Every thread owns one accumulator set per group slot in shared memory (conflict-free:
// lane t always hits the same banks whatever its slot).  Fields per (slot, thread):
//   count       u32   (rows per thread < 2^32)
//   SUM of COL  i64   (fast path: the value fits int32, so < 2^32 of them fit)
//   SUM product 96-bit = u64 lo + u32 hi (fast-path products < 2^62)
//   SUM fp64    double
//   MIN / MAX   order-encoded u32 of the int32 value (int) / u64 of the double (fp64),
//               updated with max(), so the zeroed record is the identity
constexpr int kPrivThreads = 256;
constexpr int kPrivSlots = 4;

template <class S>
struct Acc {
  __host__ __device__ static constexpr bool is_nar(uint32_t o) {
    return !S::F64 && vx_kind(o) == VX_COL && (vx_flags(o) & VS_SUM);
  }
  __host__ __device__ static constexpr bool is_wide(uint32_t o) {
    return !S::F64 && vx_kind(o) != VX_COL && (vx_flags(o) & VS_SUM);
  }
  __host__ __device__ static constexpr bool is_dbl(uint32_t o) { return S::F64 && (vx_flags(o) & VS_SUM); }
  __host__ __device__ static constexpr int nmm_of(uint32_t o) {
    return ((vx_flags(o) & VS_MIN) ? 1 : 0) + ((vx_flags(o) & VS_MAX) ? 1 : 0);
  }
  __host__ __device__ static constexpr int nar_idx(int v) {
    int c = 0;
    for (int i = 0; i < v; ++i) c += is_nar(S::OP(i)) ? 1 : 0;
    return c;
  }
  __host__ __device__ static constexpr int wide_idx(int v) {
    int c = 0;
    for (int i = 0; i < v; ++i) c += is_wide(S::OP(i)) ? 1 : 0;
    return c;
  }
  __host__ __device__ static constexpr int dbl_idx(int v) {
    int c = 0;
    for (int i = 0; i < v; ++i) c += is_dbl(S::OP(i)) ? 1 : 0;
    return c;
  }
  __host__ __device__ static constexpr int mm_before(int v) {
    int c = 0;
    for (int i = 0; i < v; ++i) c += nmm_of(S::OP(i));
    return c;
  }
  static constexpr int NNAR = nar_idx(S::NV);
  static constexpr int NWIDE = wide_idx(S::NV);
  static constexpr int NDBL = dbl_idx(S::NV);
  static constexpr int NMM = mm_before(S::NV);
  static constexpr int NMM64 = S::F64 ? NMM : 0;
  static constexpr int NMM32 = S::F64 ? 0 : NMM;
  // mm field index of value v's MIN (which = 0) or MAX (which = 1)
  __host__ __device__ static constexpr int mm_idx(int v, int which) {
    return mm_before(v) + ((which == 1 && (vx_flags(S::OP(v)) & VS_MIN)) ? 1 : 0);
  }
  // Slot-major layout: slot s owns slot_bytes(T) bytes; inside it one T-thread array per
  // field: [count u32][narrow i64 x NNAR][wide lo u64 x NWIDE][fp64 x NDBL][mm u64 x NMM64]
  // [wide hi u32 x NWIDE][mm u32 x NMM32].  A row addresses every field from two per-row
  // bases (slot base + 4*tid, slot base + 8*tid) plus compile-time offsets.
  __host__ __device__ static constexpr size_t slot_bytes(int T) {
    return ((size_t)T * (4 + 8 * (NNAR + NWIDE + NDBL + NMM64) + 4 * (NWIDE + NMM32)) + 15) / 16 * 16;
  }
  __host__ __device__ static constexpr int f_nar(int i, int T) { return 4 * T + 8 * T * i; }
  __host__ __device__ static constexpr int f_wlo(int i, int T) { return 4 * T + 8 * T * (NNAR + i); }
  __host__ __device__ static constexpr int f_dbl(int i, int T) { return 4 * T + 8 * T * (NNAR + NWIDE + i); }
  __host__ __device__ static constexpr int f_mm64(int i, int T) { return 4 * T + 8 * T * (NNAR + NWIDE + NDBL + i); }
  __host__ __device__ static constexpr int f_whi(int i, int T) {
    return 4 * T + 8 * T * (NNAR + NWIDE + NDBL + NMM64) + 4 * T * i;
  }
  __host__ __device__ static constexpr int f_mm32(int i, int T) { return f_whi(NWIDE, T) + 4 * T * i; }
  // L slots plus the trash record of the integer pair update
  __host__ __device__ static constexpr size_t bytes(int L, int T) { return (size_t)(L + (S::F64 ? 0 : 1)) * slot_bytes(T); }
  // flush fields: count, then per value SUM / MIN / MAX as flagged
  static constexpr int NF = 1 + NNAR + NWIDE + NDBL + NMM;
  // field f -> (kind: 0 count, 1 sum, 2 min, 3 max) | v << 2
  __host__ __device__ static constexpr int field(int f) {
    if (f == 0) return 0;
    int i = 1;
    for (int v = 0; v < S::NV; ++v) {
      const uint32_t fl = vx_flags(S::OP(v));
      if (fl & VS_SUM) { if (i == f) return 1 | (v << 2); ++i; }
      if (fl & VS_MIN) { if (i == f) return 2 | (v << 2); ++i; }
      if (fl & VS_MAX) { if (i == f) return 3 | (v << 2); ++i; }
    }
    return -1;
  }
};

template <class S>
__device__ __forceinline__ bool spec_is_special(KeyT<S> k) {
  if constexpr (S::NARROW_KEY) return false;
  else return k == (KeyT<S>)~0ULL;   // never placed in a slot (64-bit key ~0, or 32-bit sentinel)
}

// fp64 records: one row at a time (divergent: only rows that accumulate).
template <class S, int L, int T>
__device__ __forceinline__ void priv_add_f64(uint8_t* sm, int slot, int tid, const SRow<S>& x) {
  using A = Acc<S>;
  uint8_t* b = sm + (size_t)slot * A::slot_bytes(T);
  *(uint32_t*)(b + 4 * tid) += 1u;
#pragma unroll
  for (int v = 0; v < S::NV; ++v) {
    if constexpr (A::NDBL > 0)
      if (S::has(v, VS_SUM)) *(double*)(b + 8 * tid + A::f_dbl(A::dbl_idx(v), T)) += x.vd[v];
    if (S::has(v, VS_MIN)) {
      uint64_t* m = (uint64_t*)(b + 8 * tid + A::f_mm64(A::mm_idx(v, 0), T));
      *m = max(*m, enc_min_f(x.vd[v]));
    }
    if (S::has(v, VS_MAX)) {
      uint64_t* m = (uint64_t*)(b + 8 * tid + A::f_mm64(A::mm_idx(v, 1), T));
      *m = max(*m, enc_max_f(x.vd[v]));
    }
  }
}

__device__ __forceinline__ void add96(uint64_t& l, uint32_t& h, int64_t v) {
  uint32_t l0 = (uint32_t)l, l1 = (uint32_t)(l >> 32);
  asm("add.cc.u32 %0, %0, %3;\n\taddc.cc.u32 %1, %1, %4;\n\taddc.u32 %2, %2, %5;"
      : "+r"(l0), "+r"(l1), "+r"(h)
      : "r"((uint32_t)(uint64_t)v), "r"((uint32_t)((uint64_t)v >> 32)), "r"((uint32_t)(v >> 63)));
  l = (uint64_t)l0 | ((uint64_t)l1 << 32);
}

// Integer records: both rows of a lane in one read-modify-write pass.  Rows that do
// not accumulate here go to a trash record (slot L, never read), so the pass has no
// masking and no divergence.  Both records are loaded before either is stored — a
// pair costs one shared-memory round trip instead of two dependent ones; when both
// rows hit the same slot the second update starts from the first one's result and
// its store overwrites the first.
template <class S, int L, int T>
__device__ __forceinline__ void priv_add2(uint8_t* sm, int s0, int s1, bool g0, bool g1, int tid, const SRow<S>& x0,
                                          const SRow<S>& x1) {
  using A = Acc<S>;
  constexpr int NN = A::NNAR > 0 ? A::NNAR : 1, NW = A::NWIDE > 0 ? A::NWIDE : 1, NM = A::NMM32 > 0 ? A::NMM32 : 1;
  s0 = g0 ? s0 : L;
  s1 = g1 ? s1 : L;
  const bool same = s0 == s1;
  uint8_t* b0 = sm + (size_t)s0 * A::slot_bytes(T);
  uint8_t* b1 = sm + (size_t)s1 * A::slot_bytes(T);
  uint32_t* c0p = (uint32_t*)(b0 + 4 * tid);
  uint32_t* c1p = (uint32_t*)(b1 + 4 * tid);
  // loads
  const uint32_t c0 = *c0p, c1 = *c1p;
  int64_t n0[NN], n1[NN];
  uint64_t wl0[NW], wl1[NW];
  uint32_t wh0[NW], wh1[NW], m0[NM], m1[NM];
#pragma unroll
  for (int i = 0; i < A::NNAR; ++i) {
    n0[i] = *(const int64_t*)(b0 + 8 * tid + A::f_nar(i, T));
    n1[i] = *(const int64_t*)(b1 + 8 * tid + A::f_nar(i, T));
  }
#pragma unroll
  for (int i = 0; i < A::NWIDE; ++i) {
    wl0[i] = *(const uint64_t*)(b0 + 8 * tid + A::f_wlo(i, T));
    wl1[i] = *(const uint64_t*)(b1 + 8 * tid + A::f_wlo(i, T));
    wh0[i] = *(const uint32_t*)(b0 + 4 * tid + A::f_whi(i, T));
    wh1[i] = *(const uint32_t*)(b1 + 4 * tid + A::f_whi(i, T));
  }
#pragma unroll
  for (int i = 0; i < A::NMM32; ++i) {
    m0[i] = *(const uint32_t*)(b0 + 4 * tid + A::f_mm32(i, T));
    m1[i] = *(const uint32_t*)(b1 + 4 * tid + A::f_mm32(i, T));
  }
  // arithmetic: record 1 continues from record 0 when both are the same slot
  const uint32_t cn0 = c0 + 1u;
  const uint32_t cn1 = (same ? cn0 : c1) + 1u;
#pragma unroll
  for (int v = 0; v < S::NV; ++v) {
    if (S::has(v, VS_SUM)) {
      if (vx_kind(S::OP(v)) == VX_COL) {
        const int i = A::nar_idx(v);
        n0[i] += (int64_t)(int32_t)x0.vi[v];
        n1[i] = (same ? n0[i] : n1[i]) + (int64_t)(int32_t)x1.vi[v];
      } else {
        const int i = A::wide_idx(v);
        add96(wl0[i], wh0[i], x0.vi[v]);
        if (same) {
          wl1[i] = wl0[i];
          wh1[i] = wh0[i];
        }
        add96(wl1[i], wh1[i], x1.vi[v]);
      }
    }
    if (S::has(v, VS_MIN)) {
      const int i = A::mm_idx(v, 0);
      m0[i] = max(m0[i], s_enc32_min((int32_t)x0.vi[v]));
      m1[i] = max(same ? m0[i] : m1[i], s_enc32_min((int32_t)x1.vi[v]));
    }
    if (S::has(v, VS_MAX)) {
      const int i = A::mm_idx(v, 1);
      m0[i] = max(m0[i], s_enc32_max((int32_t)x0.vi[v]));
      m1[i] = max(same ? m0[i] : m1[i], s_enc32_max((int32_t)x1.vi[v]));
    }
  }
  // stores (record 1 last)
  *c0p = cn0;
#pragma unroll
  for (int i = 0; i < A::NNAR; ++i) *(int64_t*)(b0 + 8 * tid + A::f_nar(i, T)) = n0[i];
#pragma unroll
  for (int i = 0; i < A::NWIDE; ++i) {
    *(uint64_t*)(b0 + 8 * tid + A::f_wlo(i, T)) = wl0[i];
    *(uint32_t*)(b0 + 4 * tid + A::f_whi(i, T)) = wh0[i];
  }
#pragma unroll
  for (int i = 0; i < A::NMM32; ++i) *(uint32_t*)(b0 + 4 * tid + A::f_mm32(i, T)) = m0[i];
  *c1p = cn1;
#pragma unroll
  for (int i = 0; i < A::NNAR; ++i) *(int64_t*)(b1 + 8 * tid + A::f_nar(i, T)) = n1[i];
#pragma unroll
  for (int i = 0; i < A::NWIDE; ++i) {
    *(uint64_t*)(b1 + 8 * tid + A::f_wlo(i, T)) = wl1[i];
    *(uint32_t*)(b1 + 4 * tid + A::f_whi(i, T)) = wh1[i];
  }
#pragma unroll
  for (int i = 0; i < A::NMM32; ++i) *(uint32_t*)(b1 + 4 * tid + A::f_mm32(i, T)) = m1[i];
}

// ------------------------------------------------------------------ slot lookup
// The slot keys are cached in registers (rk); a key new to the CTA is claimed in the
// shared directory `dir` (64-bit CAS), then rk is refreshed.
template <int L>
struct DirState {
  uint64_t* dir;      // the L slot keys (~key, 0 = free)
};

// Slot of a row; resolves the rare cases (a key new to this CTA; a slow value or a key
// beyond the slots -> exact per-row update of the HBM table).  Returns true iff the row
// accumulates in private slot `slot`.
template <class S, int L>
__device__ __forceinline__ bool priv_slot(const SpecPlan& p, const DirState<L>& d, KeyT<S> (&rk)[L],
                                          const SRow<S>& x, int64_t r, int& slot) {
  static_assert(L <= 4, "slot keys are compared in registers");
  const bool special = spec_is_special<S>(x.key);
  slot = -1;
#pragma unroll
  for (int s = L - 1; s >= 0; --s)
    if (x.key == rk[s]) slot = s;
  bool go = x.q && x.fast && slot >= 0 && !special;
  if (x.q && !go) {                                   // rare: new key in this CTA, or slow value
    slot = (x.fast && !special) ? dir_find_or_insert<L>(d.dir, (uint64_t)x.key) : -1;
    if (slot >= 0) {
#pragma unroll
      for (int s = 0; s < L; ++s) {
        uint64_t sk = *(volatile uint64_t*)&d.dir[s];
        rk[s] = sk ? (KeyT<S>)~sk : (KeyT<S>)~0ULL;
      }
      go = true;
    } else {                                          // slow value, key ~0, or no slot left
      uint8_t* e = table_find_or_insert(p.g.table, p.g.mask, p.g.stride, (uint64_t)x.key, p.g.status);
      if (e) update_entry_slow(p.g, e, r);
    }
  }
  return go;
}

// Both rows (r, r + 1) of a lane.
template <class S, int L, int T>
__device__ __forceinline__ void priv_rows(const SpecPlan& p, const DirState<L>& d, KeyT<S> (&rk)[L], uint8_t* sm,
                                          int tid, const SRow<S>& x0, const SRow<S>& x1, int64_t r) {
  int s0, s1;
  const bool g0 = priv_slot<S, L>(p, d, rk, x0, r, s0);
  const bool g1 = priv_slot<S, L>(p, d, rk, x1, r + 1, s1);
  if constexpr (S::F64) {
    if (g0) priv_add_f64<S, L, T>(sm, s0, tid, x0);
    if (g1) priv_add_f64<S, L, T>(sm, s1, tid, x1);
  } else {
    priv_add2<S, L, T>(sm, s0, s1, g0, g1, tid, x0, x1);
  }
}

template <class S>
__device__ __forceinline__ void spec_row_scalar(const SpecPlan& p, int64_t r, SRow<S>& x) {
  x.fast = true;
  x.q = r < p.g.n;
  x.key = 0;
  if (!x.q) return;
  if constexpr (S::PW > 0) x.q = spec_pred<S>(p, ld1<S::PW>(p.pcol, r));
  uint64_t k0 = 0, k1 = 0;
  if constexpr (S::K0W > 0) k0 = ld1<S::K0W>(p.k0, r);
  if constexpr (S::K1W > 0) k1 = ld1<S::K1W>(p.k1, r);
  x.key = spec_key<S>(k0, k1);
  uint64_t c[S::NC];
#pragma unroll
  for (int i = 0; i < S::NC; ++i) c[i] = ld1<8>(p.col[i], r);
  spec_values<S>(p, c, x);
}

// Flush: the CTA's T private records of every (slot, field) are reduced in parallel --
// Q threads per (slot, field), each over T/Q records, then Q-lane shuffles -- and merged
// into the slot's global entry.  (A warp-by-warp shuffle tree per (slot, field) was a
// serial chain of ~NV x 5 dependent shuffles per slot: on C1, one chunk per CTA, that
// chain was most of the kernel.)  One thread per slot resolves the entry first.
// Every thread of the CTA calls it (barriers); threads tid >= T (a producer warp) only
// take part in the barriers.
template <class S, int L, int T>
__device__ __forceinline__ void priv_flush(const SpecPlan& p, const uint8_t* sm, const DirState<L>& d, int tid) {
  using A = Acc<S>;
  constexpr int Q = 4;                     // threads per (slot, field)
  constexpr int PER = T / Q;               // records each of them sums (interleaved: j = sub + Q k,
                                           // so the Q lanes of a group read Q different banks)
  constexpr int F = A::NF;
  static_assert(T % (32 * Q) == 0 || 32 % Q == 0, "Q lanes of a group share a warp");
  __shared__ uint8_t* ent[L];
  __syncthreads();
  if (tid < L) {
    const uint64_t sk = d.dir[tid];
    ent[tid] = sk != 0 ? table_find_or_insert(p.g.table, p.g.mask, p.g.stride, ~sk, p.g.status) : nullptr;
  }
  __syncthreads();
  if (tid >= T) return;
  const int sub = tid % Q;
  const unsigned gmask = ((1u << Q) - 1) << ((tid & 31) & ~(Q - 1));
  for (int i = tid / Q; i < L * F; i += T / Q) {   // uniform within a Q group
    const int s = i / F;
    const int fd = A::field(i % F);
    const int kind = fd & 3, v = fd >> 2;
    uint8_t* e = ent[s];
    if (e == nullptr) continue;
    const uint8_t* sb = sm + (size_t)s * A::slot_bytes(T);
    if (kind == 0) {
      const uint32_t* c = (const uint32_t*)sb + sub;
      unsigned long long cw = 0;
#pragma unroll 8
      for (int j = 0; j < PER; ++j) cw += c[Q * j];
      for (int o = Q / 2; o > 0; o >>= 1) cw += __shfl_xor_sync(gmask, cw, o);
      if (sub == 0 && cw) atomicAdd((unsigned long long*)(e + 8), cw);
      continue;
    }
    if (kind >= 2) {                       // MIN / MAX: max over the encodings, then the HBM encoding
      const int mi = A::mm_idx(v, kind - 2);
      unsigned long long m = 0;
      if constexpr (S::F64) {
        const uint64_t* d64 = (const uint64_t*)(sb + A::f_mm64(mi, T)) + sub;
#pragma unroll 8
        for (int j = 0; j < PER; ++j) m = max(m, (unsigned long long)d64[Q * j]);
      } else {
        const uint32_t* d32 = (const uint32_t*)(sb + A::f_mm32(mi, T)) + sub;
        uint32_t m32 = 0;
#pragma unroll 8
        for (int j = 0; j < PER; ++j) m32 = max(m32, d32[Q * j]);
        m = m32;
      }
      for (int o = Q / 2; o > 0; o >>= 1) m = max(m, __shfl_xor_sync(gmask, m, o));
      if (sub == 0) {
        const int off = kind == 2 ? p.g.vals[v].off_min : p.g.vals[v].off_max;
        unsigned long long enc = m;        // fp64: the HBM table uses the same encodings
        if constexpr (!S::F64)
          enc = kind == 2 ? enc_min_i((int64_t)s_dec32_min((uint32_t)m)) : enc_max_i((int64_t)s_dec32_max((uint32_t)m));
        if (off >= 0) atomicMax((unsigned long long*)(e + off), enc);
      }
      continue;
    }
    const int off = p.g.vals[v].off_sum;
    if constexpr (S::F64) {
      const double* dd = (const double*)(sb + A::f_dbl(A::dbl_idx(v), T)) + sub;
      double sum = 0.0;
#pragma unroll 8
      for (int j = 0; j < PER; ++j) sum += dd[Q * j];
      for (int o = Q / 2; o > 0; o >>= 1) sum += __shfl_xor_sync(gmask, sum, o);
      if (sub == 0 && off >= 0) atomicAdd((double*)(e + off), sum);
    } else {
      I128 x{0, 0};
      if (vx_kind(S::OP(v)) == VX_COL) {
        const int64_t* dn = (const int64_t*)(sb + A::f_nar(A::nar_idx(v), T)) + sub;
#pragma unroll 8
        for (int j = 0; j < PER; ++j) x = i128_add(x, i128_from_i64(dn[Q * j]));
      } else {
        const uint64_t* lo = (const uint64_t*)(sb + A::f_wlo(A::wide_idx(v), T)) + sub;
        const uint32_t* hi = (const uint32_t*)(sb + A::f_whi(A::wide_idx(v), T)) + sub;
#pragma unroll 8
        for (int j = 0; j < PER; ++j) x = i128_add(x, I128{lo[Q * j], (uint64_t)(int64_t)(int32_t)hi[Q * j]});
      }
      for (int o = Q / 2; o > 0; o >>= 1) {
        I128 y;
        y.lo = __shfl_xor_sync(gmask, x.lo, o);
        y.hi = __shfl_xor_sync(gmask, x.hi, o);
        x = i128_add(x, y);
      }
      if (sub == 0 && off >= 0) atomic_add_i128((uint64_t*)(e + off), x.lo, x.hi);
    }
  }
}

// ------------------------------------------------------------------ CTA-table tier
// "Multiple accumulators per group, inversely proportional to the number of groups"
// (§4.1.7) as a shared-memory hash table of H = 2^hb slots per CTA; the kernel
// still supports nrep replicas (consumer warp w -> replica w % nrep) but the host policy
// (fused_spec.cu tab_policy) uses one: on B200 a replica only raised the load factor.  The
// table is stored field-major (SoA) so that the 32 lanes of an atomic instruction on 32
// different slots hit different banks: keys u64[H] (~key, 0 = empty), count u32[H], then
// per value SUM -> biased sum lo u32[H], hi u32[H] (the sum of (x + 2^31) over the rows,
// exact in 64 bits; sum = biased - count * 2^31; the carry out of lo is taken from the
// atomic's return value), MIN / MAX -> order-encoded u32[H]; all updated with native 32-bit
// shared atomics.  All-zero = empty / identity.
template <class S>
struct TabL {
  // u32 field index of count / value v's sum lo, sum hi, min, max (after the u64 keys)
  __host__ __device__ static constexpr int nfield_before(int v) {
    int o = 1;
    for (int i = 0; i < v; ++i) {
      const uint32_t f = vx_flags(S::OP(i));
      o += ((f & VS_SUM) ? 2 : 0) + ((f & VS_MIN) ? 1 : 0) + ((f & VS_MAX) ? 1 : 0);
    }
    return o;
  }
  __host__ __device__ static constexpr int f_sum(int v) { return nfield_before(v); }
  __host__ __device__ static constexpr int f_min(int v) { return nfield_before(v) + ((vx_flags(S::OP(v)) & VS_SUM) ? 2 : 0); }
  __host__ __device__ static constexpr int f_max(int v) { return f_min(v) + ((vx_flags(S::OP(v)) & VS_MIN) ? 1 : 0); }
  static constexpr int NF32 = nfield_before(S::NV);
  static constexpr int BYTES_PER_SLOT = 8 + 4 * NF32;
  // replica of H slots: keys at 0, u32 field f at 8H + 4H f
  __device__ static uint32_t* fld(uint8_t* rep, uint32_t H, int f) { return (uint32_t*)(rep + 8 * (size_t)H + 4 * (size_t)H * f); }
};

// MIN / MAX into a shared u32.  With `check`, the atomic only when the value improves on
// what the slot holds: the field only moves towards the extreme, so a stale read can cost an
// unneeded atomic but never skip a needed one; after warm-up almost no row improves, and
// equal-key lanes of a warp read one broadcast word instead of serialising on one address
// (few groups / skewed keys).  Without it, one atomic (many groups: the read is extra work).
__device__ __forceinline__ void smem_max(uint32_t* a, uint32_t e, int32_t check) {
  if (check) {
    if (e > *(volatile uint32_t*)a) atomicMax(a, e);
  } else {
    atomicMax(a, e);
  }
}

constexpr uint64_t kTabMul = 0x9E3779B97F4A7C15ULL;   // multiplicative hash: home slot = top hb bits

// A warp's replica: slot count and field arrays, resolved once per kernel (registers).
template <class S>
struct TabRef {
  uint64_t* keys;
  uint32_t* f[TabL<S>::NF32];
  uint32_t hb, mask;
};

template <class S>
__device__ __forceinline__ TabRef<S> tab_ref(uint8_t* rep, uint32_t hb) {
  TabRef<S> t;
  const uint32_t H = 1u << hb;
  t.keys = (uint64_t*)rep;
  t.hb = hb;
  t.mask = H - 1;
#pragma unroll
  for (int i = 0; i < TabL<S>::NF32; ++i) t.f[i] = TabL<S>::fld(rep, H, i);
  return t;
}

// Slot-granular linear probing from the home slot, out of line (claims): slot, or -1 when
// the table is full.
static __device__ __noinline__ int tab_find_slow(uint64_t* keys, uint32_t hb, uint64_t key) {
  const uint32_t H = 1u << hb;
  const uint64_t sk = ~key;
  uint32_t h = (uint32_t)((key * kTabMul) >> (64 - hb));
  for (uint32_t probe = 0; probe < H; ++probe) {
    uint64_t* kp = &keys[h];
    const uint64_t cur = *(volatile uint64_t*)kp;
    if (cur == sk) return (int)h;
    if (cur == 0) {
      const uint64_t prev = atomicCAS((unsigned long long*)kp, 0ULL, (unsigned long long)sk);
      if (prev == 0 || prev == sk) return (int)h;
    }
    h = (h + 1) & (H - 1);
  }
  return -1;
}

// One row position of the warp (all 32 lanes call): the row into this warp's table, or, for
// a slow value / the key ~0 / a full table, the exact HBM update.  Slot-granular linear
// probing from the home slot (the top bits of key * 2^64/phi): a home-slot hit costs one
// LDS.64 and no branch; further probes run inline, warp-uniformly, while every probed slot
// holds another key (no deletions: a present key lies before the first empty slot of its
// sequence); an empty slot means a claim, out of line.
template <class S>
__device__ __forceinline__ void tab_row(const SpecPlan& p, const TabRef<S>& t, const SRow<S>& x, int64_t r) {
  using TL = TabL<S>;
  const uint64_t k = (uint64_t)x.key;
  const uint64_t sk = ~k;
  const bool ok = x.q && x.fast && !spec_is_special<S>(x.key);
  uint32_t hh = (uint32_t)((k * kTabMul) >> (64 - t.hb));
  uint64_t c = t.keys[hh];
  int h = c == sk ? (int)hh : -1;
  if (__any_sync(0xffffffffu, ok && h < 0)) {
    bool pend = ok && h < 0 && c != 0;
    bool claim = ok && h < 0 && c == 0;
    while (__any_sync(0xffffffffu, pend)) {
      if (pend) {
        hh = (hh + 1) & t.mask;
        c = t.keys[hh];
        if (c == sk) { h = (int)hh; pend = false; }
        else if (c == 0) { claim = true; pend = false; }
      }
    }
    if (__any_sync(0xffffffffu, claim))
      if (claim) h = tab_find_slow(t.keys, t.hb, k);
  }
  if (x.q && (!ok || h < 0)) {                        // slow value, key ~0, or a full replica
    uint8_t* g = table_find_or_insert(p.g.table, p.g.mask, p.g.stride, k, p.g.status);
    if (g) update_entry_slow(p.g, g, r);
  }
  if (!ok || h < 0) return;
  atomicAdd(t.f[0] + h, 1u);
#pragma unroll
  for (int v = 0; v < S::NV; ++v) {
    const int32_t xv = (int32_t)x.vi[v];
    if (S::has(v, VS_SUM)) {                        // biased add, carry from the returned value
      const uint32_t a = (uint32_t)xv ^ 0x80000000u;
      const uint32_t old = atomicAdd(t.f[TL::f_sum(v)] + h, a);
      if (old + a < old) atomicAdd(t.f[TL::f_sum(v) + 1] + h, 1u);
    }
    if (S::has(v, VS_MIN)) smem_max(t.f[TL::f_min(v)] + h, s_enc32_min(xv), p.mm_check);
    if (S::has(v, VS_MAX)) smem_max(t.f[TL::f_max(v)] + h, s_enc32_max(xv), p.mm_check);
  }
}

// Fold every replica into the HBM table (every thread of the CTA calls it).
template <class S>
__device__ __forceinline__ void tab_flush(const SpecPlan& p, uint8_t* tab, int tid, int nthreads) {
  using TL = TabL<S>;
  __syncthreads();
  const uint32_t H = 1u << p.tab_hb;
  const uint32_t slots = (uint32_t)p.tab_nrep * H;
  for (uint32_t i = tid; i < slots; i += nthreads) {
    uint8_t* rep = tab + (size_t)(i / H) * H * TL::BYTES_PER_SLOT;
    const uint32_t h = i % H;
    const uint64_t sk = ((const uint64_t*)rep)[h];
    if (sk == 0) continue;
    const uint32_t cnt = TL::fld(rep, H, 0)[h];
    uint8_t* g = table_find_or_insert(p.g.table, p.g.mask, p.g.stride, ~sk, p.g.status);
    if (!g) continue;
    atomicAdd((unsigned long long*)(g + 8), (unsigned long long)cnt);
#pragma unroll
    for (int v = 0; v < S::NV; ++v) {
      const DevValue& d = p.g.vals[v];
      if (S::has(v, VS_SUM) && d.off_sum >= 0) {
        const uint64_t b = (uint64_t)TL::fld(rep, H, TL::f_sum(v))[h] | ((uint64_t)TL::fld(rep, H, TL::f_sum(v) + 1)[h] << 32);
        const int64_t sum = (int64_t)(b - ((uint64_t)cnt << 31));
        atomic_add_i128((uint64_t*)(g + d.off_sum), (uint64_t)sum, (uint64_t)(sum >> 63));
      }
      if (S::has(v, VS_MIN) && d.off_min >= 0)
        atomicMax((unsigned long long*)(g + d.off_min),
                  (unsigned long long)enc_min_i(s_dec32_min(TL::fld(rep, H, TL::f_min(v))[h])));
      if (S::has(v, VS_MAX) && d.off_max >= 0)
        atomicMax((unsigned long long*)(g + d.off_max),
                  (unsigned long long)enc_max_i(s_dec32_max(TL::fld(rep, H, TL::f_max(v))[h])));
    }
  }
}

// ------------------------------------------------------------------ TMA bulk pipeline
// The columns reach shared memory through the copy engine: one producer thread streams
// R-row chunks of every column with cp.async.bulk into an NS-stage ring (mbarrier
// full/empty pairs); the T consumer threads read their rows from shared memory.  Loads
// no longer occupy the consumers' issue slots or registers, and the bytes in flight per
// SM (NS stages) do not depend on where the consumer warps are in their row loop.
template <class S, int R>
struct BulkStage {
  static constexpr int OFF_P = 0;
  static constexpr int OFF_K0 = OFF_P + R * S::PW;
  static constexpr int OFF_K1 = OFF_K0 + R * S::K0W;
  static constexpr int OFF_C = OFF_K1 + R * S::K1W;
  static constexpr int BYTES = OFF_C + R * 8 * S::NC;
  static_assert(R % 64 == 0, "stage rows must be whole 64-row units");
};

template <int W>
__device__ __forceinline__ void lds2(const uint8_t* base, int j, uint64_t& x0, uint64_t& x1) {
  if constexpr (W == 1) {
    uint32_t v = *(const unsigned short*)(base + j);
    x0 = v & 0xFF;
    x1 = v >> 8;
  } else if constexpr (W == 4) {
    int2 v = *(const int2*)(base + 4 * j);
    x0 = (uint64_t)(int64_t)v.x;
    x1 = (uint64_t)(int64_t)v.y;
  } else {
    longlong2 v = *(const longlong2*)(base + 8 * j);
    x0 = (uint64_t)v.x;
    x1 = (uint64_t)v.y;
  }
}

// Shared-memory bytes of the accumulation tier: L > 0 private records; L == 0 the CTA
// tables (nrep x H slots, run time).
template <class S, int L>
__host__ __device__ constexpr size_t tier_bytes(int T, uint32_t tab_slots) {
  return L > 0 ? (Acc<S>::bytes(L, T) + 127) / 128 * 128 : ((size_t)tab_slots * TabL<S>::BYTES_PER_SLOT + 127) / 128 * 128;
}

// minimum resident CTAs per SM for the register budget: without it ptxas capped the Q1
// kernel at 72 registers and spilled two values per 64-row unit to local memory (+0.6 GB
// of L2 traffic on C4, 3.56 -> 4.19 ms); the shared-memory footprint allows 2-3 CTAs anyway
template <int T>
__host__ __device__ constexpr int bulk_min_blocks() { return T <= 128 ? 3 : (T <= 512 ? 2 : 1); }

// Select-compact-gather stages: the ring's stage buffers carry RS rows of the predicate
// column only — US 64-row units per consumer warp (at most 5: the warp keeps 2 ballot masks
// per unit in registers).
template <class S, class B, int NW>
struct SparseStage {
  static constexpr int PWB = S::PW > 0 ? S::PW : 1;
  static constexpr int FIT = B::BYTES / PWB / (64 * NW);
  static constexpr int US = FIT < 1 ? 1 : (FIT > 5 ? 5 : FIT);
  static constexpr int RS = 64 * NW * US;
  static_assert(S::PW == 0 || RS * S::PW <= B::BYTES, "sparse stage must fit a dense stage buffer");
};

// Consumers of the select-compact-gather mode (the paper's select -> prefix-sum compaction
// -> grouping, §4.1.1-4.1.2, per stage and per warp): a warp evaluates the
// predicate on its US units of kSparseBatch consecutive stages of its CTA, releasing each
// stage as soon as its ballots are taken, then turns the ballot masks (shared memory, one
// word per unit and row parity) into a compacted list of qualifying rows (n-th set bit)
// and gathers key and value columns for those rows only, 32 at a time, from global
// memory.  Batching stages doubles the gathers in flight per warp (latency-bound at 1 %).
constexpr int kSparseBatch = 2;

template <class S, int L, int LD, int T, class B, int NS>
__device__ __forceinline__ void sparse_consume(const SpecPlan& p, const DirState<LD>& d, KeyT<S> (&rk)[LD],
                                               uint8_t* sm, const TabRef<S>& mytab, const uint8_t* stg,
                                               uint64_t* full, uint64_t* empty, int64_t nfull, int tid) {
  constexpr int NW = T / 32;
  constexpr int US = SparseStage<S, B, NW>::US;
  constexpr int RS = SparseStage<S, B, NW>::RS;
  constexpr int NM = 2 * US * kSparseBatch;               // masks per warp and batch
  __shared__ uint32_t smk[NW][NM];
  const int lane = tid & 31, wid = tid >> 5;
  uint32_t* mk = smk[wid];
  int stage = 0;
  uint32_t phase = 0;
  for (int64_t c0 = blockIdx.x; c0 < nfull; c0 += (int64_t)kSparseBatch * gridDim.x) {
    int tot = 0;
#pragma unroll
    for (int g = 0; g < kSparseBatch; ++g) {
      const int64_t c = c0 + (int64_t)g * gridDim.x;
      if (c >= nfull) {                                    // (warp-uniform) no stage: empty masks
        if (lane < 2 * US) mk[g * 2 * US + lane] = 0u;
        continue;
      }
      mbar_wait_mode(&full[stage], phase, p.cwait);
      const uint8_t* sd = stg + (size_t)stage * B::BYTES;
#pragma unroll
      for (int u = 0; u < US; ++u) {
        uint64_t a0, a1;
        lds2<S::PW>(sd, (wid * US + u) * 64 + 2 * lane, a0, a1);
        const bool q0 = spec_pred<S>(p, a0), q1 = spec_pred<S>(p, a1);
        if (p.g.bitmap_out) emit_bitmap_unit(p.g, c * RS + (wid * US + u) * 64, lane, q0, q1);
        const uint32_t m0 = __ballot_sync(0xffffffffu, q0), m1 = __ballot_sync(0xffffffffu, q1);
        if (lane == 0) {
          mk[(g * US + u) * 2] = m0;
          mk[(g * US + u) * 2 + 1] = m1;
        }
        tot += __popc(m0) + __popc(m1);
      }
      mbar_release_reads(&empty[stage], lane);
      if (++stage == NS) {
        stage = 0;
        phase ^= 1;
      }
    }
    __syncwarp();
    for (int b0 = 0; b0 < tot; b0 += 32) {              // warp-uniform rounds of 32 rows
      int t = b0 + lane;
      const bool valid = t < tot;
      int64_t r = 0;                                     // the t-th qualifying row of the batch
#pragma unroll 4
      for (int m = 0; m < NM; ++m) {
        const uint32_t w = mk[m];
        const int cm = __popc(w);
        if (t >= 0 && t < cm) {
          const int g = m / (2 * US), u = (m / 2) % US;
          r = (c0 + (int64_t)g * gridDim.x) * RS + (wid * US + u) * 64 + 2 * (int)__fns(w, 0, t + 1) + (m & 1);
        }
        t -= cm;
      }
      SRow<S> x;
      x.q = valid;
      x.fast = true;
      uint64_t k0 = 0, k1 = 0, cv[S::NC];
#pragma unroll
      for (int i = 0; i < S::NC; ++i) cv[i] = 0;
      if (valid) {
        if constexpr (S::K0W > 0) k0 = ld1<S::K0W>(p.k0, r);
        if constexpr (S::K1W > 0) k1 = ld1<S::K1W>(p.k1, r);
#pragma unroll
        for (int i = 0; i < S::NC; ++i) cv[i] = ld1<8>(p.col[i], r);
      }
      x.key = spec_key<S>(k0, k1);
      spec_values<S>(p, cv, x);
      if constexpr (L > 0) {
        SRow<S> none = x;                                // second row position unused
        none.q = false;
        priv_rows<S, LD, T>(p, d, rk, sm, tid, x, none, r);
      } else {
        tab_row<S>(p, mytab, x, r);
      }
    }
    __syncwarp();                                        // masks are rewritten by the next batch
  }
}

// Select-compact-gather decision, identical in every CTA of both kernels (k_sga_sparse runs
// iff k_sga_bulk exits): the predicate on kSparseSample rows at fixed positions spread
// over the input, against p.sparse_pct %.  Every thread of the CTA calls it.
constexpr int kSparseSample = 1024;

template <class S, int NT>
__device__ __forceinline__ bool spec_sparse(const SpecPlan& p) {
  if constexpr (S::PW == 0) {
    return false;
  } else {
    constexpr int PER = (kSparseSample + NT - 1) / NT;
    __shared__ int s_cnt;
    const int64_t span = p.g.n / kSparseSample;
    int q = 0;
    if (span > 0) {
      uint64_t raw[PER];
#pragma unroll
      for (int k = 0; k < PER; ++k) {                   // all loads in flight, then the predicates
        const int i = threadIdx.x + k * NT;
        raw[k] = i < kSparseSample ? ld1<S::PW>(p.pcol, (int64_t)i * span) : 0;
      }
#pragma unroll
      for (int k = 0; k < PER; ++k) q += (threadIdx.x + k * NT < kSparseSample && spec_pred<S>(p, raw[k])) ? 1 : 0;
    }
    if (threadIdx.x == 0) s_cnt = 0;
    __syncthreads();
    if (q) atomicAdd(&s_cnt, q);
    __syncthreads();
    return span > 0 && 100 * s_cnt < p.sparse_pct * kSparseSample;
  }
}

// Shared-memory setup of both bulk kernels: zeroed accumulation tier, directory, barriers.
template <class S, int L, int T, int NS>
__device__ __forceinline__ size_t bulk_setup(const SpecPlan& p, uint8_t* sm, uint64_t* dir, uint64_t* full,
                                             uint64_t* empty, int tid) {
  constexpr int NW = T / 32;
  constexpr int LD = L > 0 ? L : 1;
  const uint32_t tab_slots = L > 0 ? 0u : ((uint32_t)p.tab_nrep << p.tab_hb);
  const size_t tb = tier_bytes<S, L>(T, tab_slots);
  {
    uint4* z = (uint4*)sm;
    for (int i = tid; i < (int)(tb / 16); i += T + 32) z[i] = make_uint4(0, 0, 0, 0);
  }
  for (int i = tid; i < LD; i += T + 32) dir[i] = 0;
  if (tid == 0) {
    for (int s = 0; s < NS; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NW);
    }
    mbar_fence_init();
  }
  __syncthreads();
  return tb;
}

// CTA-table tier: this warp's table
template <class S, int L>
__device__ __forceinline__ TabRef<S> bulk_tab(const SpecPlan& p, uint8_t* sm, int wid) {
  return tab_ref<S>(sm + (L > 0 ? 0 : (size_t)(wid % (p.tab_nrep ? p.tab_nrep : 1)) * ((size_t)1 << p.tab_hb) *
                                           TabL<S>::BYTES_PER_SLOT),
                    L > 0 ? 5u : p.tab_hb);
}

// Ragged tail (< one chunk of `crows` rows after nfull chunks): one CTA, scalar loads
// straight from global memory.
template <class S, int L, int LD, int T>
__device__ __forceinline__ void bulk_tail(const SpecPlan& p, const DirState<LD>& d, KeyT<S> (&rk)[LD], uint8_t* sm,
                                          const TabRef<S>& mytab, int64_t nfull, int64_t crows, int tid) {
  constexpr int NW = T / 32;
  const int lane = tid & 31, wid = tid >> 5;
  if (blockIdx.x != (int)(nfull % gridDim.x)) return;
  for (int64_t base = nfull * crows + (int64_t)wid * 64; base < p.g.n; base += 64 * NW) {
    const int64_t r = base + 2 * lane;
    SRow<S> x0, x1;
    spec_row_scalar<S>(p, r, x0);
    spec_row_scalar<S>(p, r + 1, x1);
    if (p.g.bitmap_out) emit_bitmap_unit(p.g, base, lane, x0.q, x1.q);
    if constexpr (L > 0) {
      priv_rows<S, LD, T>(p, d, rk, sm, tid, x0, x1, r);
    } else {
      tab_row<S>(p, mytab, x0, r);
      tab_row<S>(p, mytab, x1, r + 1);
    }
  }
}

template <class S, int L, int T, int R, int NS>
__global__ void __launch_bounds__(T + 32, bulk_min_blocks<T>()) k_sga_bulk(const __grid_constant__ SpecPlan p) {
  using B = BulkStage<S, R>;
  constexpr int NW = T / 32;                 // consumer warps
  constexpr int UPW = R / 64 / NW;           // 64-row units per consumer warp per stage
  static_assert(UPW >= 1 && UPW * 64 * NW == R, "R must be 64 * consumer warps * units");
  constexpr int LD = L > 0 ? L : 1;
  extern __shared__ __align__(128) uint8_t sm[];
  __shared__ uint64_t dir[LD];
  __shared__ __align__(8) uint64_t full[NS], empty[NS];
  const int tid = threadIdx.x, lane = tid & 31, wid = tid >> 5;
  if constexpr (S::PW > 0)
    if (p.sparse_pct > 0 && spec_sparse<S, T + 32>(p)) return;   // k_sga_sparse took this call
  uint8_t* stg = sm + bulk_setup<S, L, T, NS>(p, sm, dir, full, empty, tid);
  const DirState<LD> d{dir};
  const TabRef<S> mytab = bulk_tab<S, L>(p, sm, wid);
  const int64_t n = p.g.n;
  const int64_t nfull = n / R;
  if (wid == NW) {
    // ---- producer: one elected thread streams every column chunk of this CTA's chunks
    if (lane == 0) {
      const uint64_t pol = policy_evict_first();
      int stage = 0;
      uint32_t phase = 0;
      for (int64_t c = blockIdx.x; c < nfull; c += gridDim.x) {
        mbar_wait_mode(&empty[stage], phase ^ 1, p.pwait);
        uint64_t* fb = &full[stage];
        mbar_arrive_expect_tx(fb, B::BYTES);
        uint8_t* dst = stg + (size_t)stage * B::BYTES;
        const int64_t r0 = c * R;
        if constexpr (S::PW > 0) bulk_g2s(dst + B::OFF_P, (const uint8_t*)p.pcol + r0 * S::PW, R * S::PW, fb, pol);
        if constexpr (S::K0W > 0) bulk_g2s(dst + B::OFF_K0, (const uint8_t*)p.k0 + r0 * S::K0W, R * S::K0W, fb, pol);
        if constexpr (S::K1W > 0) bulk_g2s(dst + B::OFF_K1, (const uint8_t*)p.k1 + r0 * S::K1W, R * S::K1W, fb, pol);
#pragma unroll
        for (int i = 0; i < S::NC; ++i)
          bulk_g2s(dst + B::OFF_C + i * R * 8, (const uint8_t*)p.col[i] + r0 * 8, R * 8, fb, pol);
        if (++stage == NS) {
          stage = 0;
          phase ^= 1;
        }
      }
    }
  } else {
    // ---- consumers
    KeyT<S> rk[LD];
#pragma unroll
    for (int s = 0; s < LD; ++s) rk[s] = (KeyT<S>)~0ULL;
    int stage = 0;
    uint32_t phase = 0;
    for (int64_t c = blockIdx.x; c < nfull; c += gridDim.x) {
      mbar_wait_mode(&full[stage], phase, p.cwait);
      const uint8_t* sd = stg + (size_t)stage * B::BYTES;
      uint64_t pr[UPW][2], k0[UPW][2], k1[UPW][2], cv[UPW][2][S::NC];
#pragma unroll
      for (int u = 0; u < UPW; ++u) {
        const int j = (wid * UPW + u) * 64 + 2 * lane;
        if constexpr (S::PW > 0) lds2<S::PW>(sd + B::OFF_P, j, pr[u][0], pr[u][1]);
        if constexpr (S::K0W > 0) lds2<S::K0W>(sd + B::OFF_K0, j, k0[u][0], k0[u][1]);
        if constexpr (S::K1W > 0) lds2<S::K1W>(sd + B::OFF_K1, j, k1[u][0], k1[u][1]);
#pragma unroll
        for (int i = 0; i < S::NC; ++i) lds2<8>(sd + B::OFF_C + i * R * 8, j, cv[u][0][i], cv[u][1][i]);
      }
      mbar_release_reads(&empty[stage], lane);       // the stage's bytes are in registers now
      if (++stage == NS) {
        stage = 0;
        phase ^= 1;
      }
#pragma unroll
      for (int u = 0; u < UPW; ++u) {
        const int64_t base = c * R + (wid * UPW + u) * 64;
        const int64_t r = base + 2 * lane;
        SRow<S> x[2];
#pragma unroll
        for (int k = 0; k < 2; ++k) {
          x[k].q = true;
          if constexpr (S::PW > 0) x[k].q = spec_pred<S>(p, pr[u][k]);
          x[k].key = spec_key<S>(S::K0W ? k0[u][k] : 0, S::K1W ? k1[u][k] : 0);
          x[k].fast = true;
          spec_values<S>(p, cv[u][k], x[k]);
        }
        if (p.g.bitmap_out) emit_bitmap_unit(p.g, base, lane, x[0].q, x[1].q);
        if constexpr (L > 0) {
          priv_rows<S, LD, T>(p, d, rk, sm, tid, x[0], x[1], r);
        } else {
          tab_row<S>(p, mytab, x[0], r);
          tab_row<S>(p, mytab, x[1], r + 1);
        }
      }
    }
    bulk_tail<S, L, LD, T>(p, d, rk, sm, mytab, nfull, R, tid);
  }
  if constexpr (L > 0) priv_flush<S, LD, T>(p, sm, d, tid);
  else tab_flush<S>(p, sm, tid, T + 32);
}

// The select-compact-gather twin of k_sga_bulk (same accumulation tiers and shared-memory
// layout; launched before it, exactly one of the two runs past its sample): the ring
// carries the predicate column only, RS rows per stage, and the consumers gather key and
// value sectors for the qualifying rows (sparse_consume).
template <class S, int L, int T, int R, int NS>
__global__ void __launch_bounds__(T + 32, bulk_min_blocks<T>()) k_sga_sparse(const __grid_constant__ SpecPlan p) {
  static_assert(S::PW > 0, "select-compact-gather needs a predicate");
  using B = BulkStage<S, R>;
  constexpr int NW = T / 32;
  constexpr int RS = SparseStage<S, B, NW>::RS;
  constexpr int LD = L > 0 ? L : 1;
  extern __shared__ __align__(128) uint8_t sm[];
  __shared__ uint64_t dir[LD];
  __shared__ __align__(8) uint64_t full[NS], empty[NS];
  const int tid = threadIdx.x, lane = tid & 31, wid = tid >> 5;
  if (p.sparse_pct <= 0 || !spec_sparse<S, T + 32>(p)) return;   // k_sga_bulk takes this call
  uint8_t* stg = sm + bulk_setup<S, L, T, NS>(p, sm, dir, full, empty, tid);
  const DirState<LD> d{dir};
  const TabRef<S> mytab = bulk_tab<S, L>(p, sm, wid);
  const int64_t nfull = p.g.n / RS;
  if (wid == NW) {
    if (lane == 0) {
      const uint64_t pol = policy_evict_first();
      int stage = 0;
      uint32_t phase = 0;
      for (int64_t c = blockIdx.x; c < nfull; c += gridDim.x) {
        mbar_wait_mode(&empty[stage], phase ^ 1, p.pwait);
        uint64_t* fb = &full[stage];
        mbar_arrive_expect_tx(fb, RS * S::PW);
        bulk_g2s(stg + (size_t)stage * B::BYTES, (const uint8_t*)p.pcol + c * RS * S::PW, RS * S::PW, fb, pol);
        if (++stage == NS) {
          stage = 0;
          phase ^= 1;
        }
      }
    }
  } else {
    KeyT<S> rk[LD];
#pragma unroll
    for (int s = 0; s < LD; ++s) rk[s] = (KeyT<S>)~0ULL;
    sparse_consume<S, L, LD, T, B, NS>(p, d, rk, sm, mytab, stg, full, empty, nfull, tid);
    bulk_tail<S, L, LD, T>(p, d, rk, sm, mytab, nfull, RS, tid);
  }
  if constexpr (L > 0) priv_flush<S, LD, T>(p, sm, d, tid);
  else tab_flush<S>(p, sm, tid, T + 32);
}

template <class S, int L>
__global__ void __launch_bounds__(kPrivThreads) k_sga_priv(const __grid_constant__ SpecPlan p) {
  using A = Acc<S>;
  constexpr int T = kPrivThreads;
  extern __shared__ __align__(16) uint8_t sm[];
  __shared__ uint64_t dir[L];
  const int tid = threadIdx.x, lane = tid & 31;
  {
    uint4* z = (uint4*)sm;
    for (int i = tid; i < (int)(A::bytes(L, T) / 16); i += T) z[i] = make_uint4(0, 0, 0, 0);
  }
  if (tid < L) dir[tid] = 0;
  __syncthreads();
  const DirState<L> d{dir};
  KeyT<S> rk[L];
#pragma unroll
  for (int s = 0; s < L; ++s) rk[s] = (KeyT<S>)~0ULL;

  constexpr int U = 2;
  constexpr int kTile = 64 * U;
  const int64_t warp = (blockIdx.x * (int64_t)T + tid) >> 5;
  const int64_t nwarps = ((int64_t)gridDim.x * T) >> 5;
  const int64_t n = p.g.n;
  const int64_t ntiles = (n + kTile - 1) / kTile;
  for (int64_t t = warp; t < ntiles; t += nwarps) {
    const int64_t base = t * kTile;
    if (base + kTile <= n) {
      uint64_t pr[U][2], k0[U][2], k1[U][2], c[U][2][S::NC];
#pragma unroll
      for (int u = 0; u < U; ++u) {
        const int64_t r = base + 64 * u + 2 * lane;
        if constexpr (S::PW > 0) ld2<S::PW>(p.pcol, r, pr[u][0], pr[u][1]);
        if constexpr (S::K0W > 0) ld2<S::K0W>(p.k0, r, k0[u][0], k0[u][1]);
        if constexpr (S::K1W > 0) ld2<S::K1W>(p.k1, r, k1[u][0], k1[u][1]);
#pragma unroll
        for (int i = 0; i < S::NC; ++i) ld2<8>(p.col[i], r, c[u][0][i], c[u][1][i]);
      }
#pragma unroll
      for (int u = 0; u < U; ++u) {
        const int64_t r = base + 64 * u + 2 * lane;
        SRow<S> x[2];
#pragma unroll
        for (int k = 0; k < 2; ++k) {
          x[k].q = true;
          if constexpr (S::PW > 0) x[k].q = spec_pred<S>(p, pr[u][k]);
          x[k].key = spec_key<S>(S::K0W ? k0[u][k] : 0, S::K1W ? k1[u][k] : 0);
          x[k].fast = true;
          spec_values<S>(p, c[u][k], x[k]);
        }
        if (p.g.bitmap_out) emit_bitmap_unit(p.g, base + 64 * u, lane, x[0].q, x[1].q);
        priv_rows<S, L, T>(p, d, rk, sm, tid, x[0], x[1], r);
      }
    } else {
      for (int u = 0; u < U; ++u) {
        const int64_t r = base + 64 * u + 2 * lane;
        SRow<S> x0, x1;
        spec_row_scalar<S>(p, r, x0);
        spec_row_scalar<S>(p, r + 1, x1);
        if (p.g.bitmap_out) emit_bitmap_unit(p.g, base + 64 * u, lane, x0.q, x1.q);
        priv_rows<S, L, T>(p, d, rk, sm, tid, x0, x1, r);
      }
    }
  }
  priv_flush<S, L, T>(p, sm, d, tid);
}

}  // namespace ocl
