// fused_spec.cu — the TPC-H Q1-signature fused kernel (few groups; SUM / COUNT /
// AVG over a predicate column, two u8 key columns and int64 / fp64 decimals).
//
// Same method, semantics and accumulation scheme as the unified kernel in fused.cu
// (§4.1.1 selection, §4.1.6 grouping, §4.1.7 aggregation; private
// per-thread accumulators in shared memory), specialised by hand for the
// Q1 plan shape: accumulator arrays grouped by type ([type][slot][value][thread]),
// narrow sums in 64 bits, products in 96 bits, compile-time layout and key packing.
// Two kernels: k_sga_priv loads the columns into registers (vector LDG, two units in
// flight per warp); k_sga_bulk (default) streams them into shared memory with TMA
// bulk copies (cp.async.bulk + mbarrier ring, one producer warp) so the consumer
// warps only compute.  On B200 C4 (600M rows) k_sga_bulk runs in ~3.45 ms
// (~6.6 TB/s, ~101 % of the measured copy bandwidth); the generic StaticShape
// instantiation of k_sga takes 5.1-5.5 ms.  launch_fused (fused.cu)
// tries these kernels first for few-group plans; OCL_NO_SPEC=1 disables them.
#include <type_traits>

#include "bulk.cuh"
#include "launch.cuh"
#include "rowops.cuh"

namespace ocl {

enum : uint32_t { VX_COL = 0, VX_M1 = 1, VX_M1P = 2 };
__host__ __device__ constexpr uint32_t vop(uint32_t kind, uint32_t a, uint32_t b = 0, uint32_t c = 0) {
  return kind | (a << 2) | (b << 5) | (c << 8);
}
__host__ __device__ constexpr uint32_t vx_kind(uint32_t o) { return o & 3; }
__host__ __device__ constexpr uint32_t vx_a(uint32_t o) { return (o >> 2) & 7; }
__host__ __device__ constexpr uint32_t vx_b(uint32_t o) { return (o >> 5) & 7; }
__host__ __device__ constexpr uint32_t vx_c(uint32_t o) { return (o >> 8) & 7; }

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
};

struct SpecPlan {
  Plan g;                     // generic plan (slow path, tail rows, flush offsets)
  const void* pcol;
  int32_t plo, phi;           // predicate bounds clamped to int32 (int columns)
  const void* k0;
  const void* k1;
  const void* col[4];
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

template <class S>
using KeyT = typename std::conditional<(S::KBITS <= 32), uint32_t, uint64_t>::type;

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
// Low-G tier: every thread owns one accumulator set per group slot in shared memory
// (conflict-free: lane t always hits the same banks whatever its slot).  A row costs
// one slot-indexed read-modify-write per accumulator — no atomics, no per-slot
// predication — the limit of the paper's "multiple accumulators per group" in local
// memory.
//   count      u32   (rows per thread < 2^32)
//   COL value  i64   (fast path: the value fits int32, so < 2^32 of them fit)
//   product    96-bit = u64 lo + u32 hi (fast-path products < 2^62)
//   fp64       double
constexpr int kPrivThreads = 256;
constexpr int kPrivSlots = 4;

template <class S>
struct Acc {
  static constexpr int nnar() {
    int c = 0;
    for (int v = 0; v < S::NV; ++v) c += vx_kind(S::OP(v)) == VX_COL ? 1 : 0;
    return c;
  }
  static constexpr int NNAR = S::F64 ? 0 : nnar();
  static constexpr int NWIDE = S::F64 ? 0 : S::NV - nnar();
  static constexpr int NDBL = S::F64 ? S::NV : 0;
  __host__ __device__ static constexpr int nar_idx(int v) {
    int c = 0;
    for (int i = 0; i < v; ++i) c += vx_kind(S::OP(i)) == VX_COL ? 1 : 0;
    return c;
  }
  __host__ __device__ static constexpr int wide_idx(int v) { return v - nar_idx(v); }
  // Slot-major layout: slot s owns slot_bytes(T) bytes; inside it one T-thread array
  // per field: [count u32][narrow i64 x NNAR][wide lo u64 x NWIDE][fp64 x NDBL]
  // [wide hi u32 x NWIDE].  A row addresses every field from two per-row bases
  // (slot base + 4*tid, slot base + 8*tid) plus compile-time offsets.
  __host__ __device__ static constexpr size_t slot_bytes(int T) {
    return ((size_t)T * (4 + 8 * NNAR + 12 * NWIDE + 8 * NDBL) + 15) / 16 * 16;
  }
  __host__ __device__ static constexpr int f_nar(int i, int T) { return 4 * T + 8 * T * i; }
  __host__ __device__ static constexpr int f_wlo(int i, int T) { return 4 * T + 8 * T * (NNAR + i); }
  __host__ __device__ static constexpr int f_dbl(int i, int T) { return 4 * T + 8 * T * (NNAR + NWIDE + i); }
  __host__ __device__ static constexpr int f_whi(int i, int T) { return 4 * T + 8 * T * (NNAR + NWIDE + NDBL) + 4 * T * i; }
  // L slots plus the trash record of the integer pair update
  __host__ __device__ static constexpr size_t bytes(int L, int T) { return (size_t)(L + (S::F64 ? 0 : 1)) * slot_bytes(T); }
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
  for (int v = 0; v < S::NV; ++v) *(double*)(b + 8 * tid + A::f_dbl(v, T)) += x.vd[v];
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
  constexpr int NN = A::NNAR > 0 ? A::NNAR : 1, NW = A::NWIDE > 0 ? A::NWIDE : 1;
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
  uint32_t wh0[NW], wh1[NW];
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
  // arithmetic: record 1 continues from record 0 when both are the same slot
  const uint32_t cn0 = c0 + 1u;
  const uint32_t cn1 = (same ? cn0 : c1) + 1u;
#pragma unroll
  for (int v = 0; v < S::NV; ++v) {
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
  // stores (record 1 last)
  *c0p = cn0;
#pragma unroll
  for (int i = 0; i < A::NNAR; ++i) *(int64_t*)(b0 + 8 * tid + A::f_nar(i, T)) = n0[i];
#pragma unroll
  for (int i = 0; i < A::NWIDE; ++i) {
    *(uint64_t*)(b0 + 8 * tid + A::f_wlo(i, T)) = wl0[i];
    *(uint32_t*)(b0 + 4 * tid + A::f_whi(i, T)) = wh0[i];
  }
  *c1p = cn1;
#pragma unroll
  for (int i = 0; i < A::NNAR; ++i) *(int64_t*)(b1 + 8 * tid + A::f_nar(i, T)) = n1[i];
#pragma unroll
  for (int i = 0; i < A::NWIDE; ++i) {
    *(uint64_t*)(b1 + 8 * tid + A::f_wlo(i, T)) = wl1[i];
    *(uint32_t*)(b1 + 4 * tid + A::f_whi(i, T)) = wh1[i];
  }
}

// Slot of a row; resolves the rare cases (a key new to this CTA -> directory insert;
// a slow value or a key beyond the slots -> exact per-row update of the HBM table).
// Returns true iff the row accumulates in private slot `slot`.
template <class S, int L>
__device__ __forceinline__ bool priv_slot(const SpecPlan& p, uint64_t* dir, KeyT<S> (&rk)[L], const SRow<S>& x,
                                          int64_t r, int& slot) {
  slot = -1;
#pragma unroll
  for (int s = L - 1; s >= 0; --s)
    if (x.key == rk[s]) slot = s;
  const bool special = spec_is_special<S>(x.key);
  bool go = x.q && x.fast && slot >= 0 && !special;
  if (x.q && !go) {                                    // rare: new key in this CTA, or slow value
    slot = (x.fast && !special) ? dir_find_or_insert<L>(dir, (uint64_t)x.key) : -1;
    if (slot >= 0) {
#pragma unroll
      for (int s = 0; s < L; ++s) {
        uint64_t sk = *(volatile uint64_t*)&dir[s];
        rk[s] = sk ? (KeyT<S>)~sk : (KeyT<S>)~0ULL;
      }
      go = true;
    } else {
      uint8_t* e = table_find_or_insert(p.g.table, p.g.mask, p.g.stride, (uint64_t)x.key, p.g.status);
      if (e) update_entry_slow(p.g, e, r);
    }
  }
  return go;
}

// Both rows (r, r + 1) of a lane.
template <class S, int L, int T = kPrivThreads>
__device__ __forceinline__ void priv_rows(const SpecPlan& p, uint64_t* dir, KeyT<S> (&rk)[L], uint8_t* sm, int tid,
                                          const SRow<S>& x0, const SRow<S>& x1, int64_t r) {
  int s0, s1;
  const bool g0 = priv_slot<S, L>(p, dir, rk, x0, r, s0);
  const bool g1 = priv_slot<S, L>(p, dir, rk, x1, r + 1, s1);
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

// Flush: the CTA's T private records of every (slot, field) are summed in parallel --
// Q threads per (slot, field), each over T/Q records, then Q-lane shuffles -- and added
// into the slot's global entry.  (A warp-by-warp shuffle tree per (slot, field) was a
// serial chain of ~NV x 5 dependent shuffles per slot: on C1, one chunk per CTA, that
// chain was most of the kernel.)  One thread per slot resolves the entry first.
// Every thread of the CTA calls it (barriers); threads tid >= T (a producer warp) only
// take part in the barriers.
template <class S, int L, int T>
__device__ __forceinline__ void priv_flush(const SpecPlan& p, const uint8_t* sm, const uint64_t* dir, int tid) {
  using A = Acc<S>;
  constexpr int Q = 4;                     // threads per (slot, field)
  constexpr int PER = T / Q;               // records each of them sums (interleaved: j = sub + Q k,
                                           // so the Q lanes of a group read Q different banks)
  constexpr int F = 1 + S::NV;             // COUNT + the value sums
  static_assert(T % (32 * Q) == 0 || 32 % Q == 0, "Q lanes of a group share a warp");
  __shared__ uint8_t* ent[L];
  __syncthreads();
  if (tid < L) {
    const uint64_t sk = dir[tid];
    ent[tid] = sk != 0 ? table_find_or_insert(p.g.table, p.g.mask, p.g.stride, ~sk, p.g.status) : nullptr;
  }
  __syncthreads();
  if (tid >= T) return;
  const int sub = tid % Q;
  const unsigned gmask = ((1u << Q) - 1) << ((tid & 31) & ~(Q - 1));
  for (int i = tid / Q; i < L * F; i += T / Q) {   // uniform within a Q group
    const int s = i / F, v = i % F - 1;
    uint8_t* e = ent[s];
    if (e == nullptr) continue;
    const uint8_t* sb = sm + (size_t)s * A::slot_bytes(T);
        if (v < 0) {
      const uint32_t* c = (const uint32_t*)sb + sub;
      unsigned long long cw = 0;
#pragma unroll 8
      for (int j = 0; j < PER; ++j) cw += c[Q * j];
      for (int o = Q / 2; o > 0; o >>= 1) cw += __shfl_xor_sync(gmask, cw, o);
      if (sub == 0 && cw) atomicAdd((unsigned long long*)(e + 8), cw);
      continue;
    }
    const int off = p.g.vals[v].off_sum;
    if constexpr (S::F64) {
      const double* d = (const double*)(sb + A::f_dbl(v, T)) + sub;
      double sum = 0.0;
#pragma unroll 8
      for (int j = 0; j < PER; ++j) sum += d[Q * j];
      for (int o = Q / 2; o > 0; o >>= 1) sum += __shfl_xor_sync(gmask, sum, o);
      if (sub == 0 && off >= 0) atomicAdd((double*)(e + off), sum);
    } else {
      I128 x{0, 0};
      if (vx_kind(S::OP(v)) == VX_COL) {
        const int64_t* d = (const int64_t*)(sb + A::f_nar(A::nar_idx(v), T)) + sub;
#pragma unroll 8
        for (int j = 0; j < PER; ++j) x = i128_add(x, i128_from_i64(d[Q * j]));
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

// ------------------------------------------------------------------ TMA bulk pipeline
// Same rows, semantics and accumulators as k_sga_priv, but the columns reach shared
// memory through the copy engine: one producer thread streams R-row chunks of every
// column with cp.async.bulk into an NS-stage ring (mbarrier full/empty pairs); the T
// consumer threads read their rows from shared memory.  Loads no longer occupy the
// consumers' issue slots or registers, and the bytes in flight per SM (NS stages) do
// not depend on where the consumer warps are in their row loop.
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

template <class S>
__host__ __device__ constexpr size_t bulk_acc_bytes(int L, int T) {
  return (Acc<S>::bytes(L, T) + 127) / 128 * 128;
}

template <class S, int L, int T, int R, int NS>
__global__ void __launch_bounds__(T + 32) k_sga_bulk(const __grid_constant__ SpecPlan p) {
  using A = Acc<S>;
  using B = BulkStage<S, R>;
  constexpr int NW = T / 32;                 // consumer warps
  constexpr int UPW = R / 64 / NW;           // 64-row units per consumer warp per stage
  static_assert(UPW >= 1 && UPW * 64 * NW == R, "R must be 64 * consumer warps * units");
  extern __shared__ __align__(128) uint8_t sm[];
  uint8_t* stg = sm + bulk_acc_bytes<S>(L, T);
  __shared__ uint64_t dir[L];
  __shared__ __align__(8) uint64_t full[NS], empty[NS];
  const int tid = threadIdx.x, lane = tid & 31, wid = tid >> 5;
  {
    uint4* z = (uint4*)sm;
    for (int i = tid; i < (int)(A::bytes(L, T) / 16); i += T + 32) z[i] = make_uint4(0, 0, 0, 0);
  }
  if (tid < L) dir[tid] = 0;
  if (tid == 0) {
    for (int s = 0; s < NS; ++s) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], NW);
    }
    mbar_fence_init();
  }
  __syncthreads();
  const int64_t n = p.g.n;
  const int64_t nfull = n / R;
  if (wid == NW) {
    // ---- producer: one elected thread streams every column chunk of this CTA's chunks
    if (lane == 0) {
      const uint64_t pol = policy_evict_first();
      int stage = 0;
      uint32_t phase = 0;
      for (int64_t c = blockIdx.x; c < nfull; c += gridDim.x) {
        mbar_wait(&empty[stage], phase ^ 1);
        uint64_t* fb = &full[stage];
        mbar_arrive_expect_tx(fb, B::BYTES);
        uint8_t* d = stg + (size_t)stage * B::BYTES;
        const int64_t r0 = c * R;
        if constexpr (S::PW > 0) bulk_g2s(d + B::OFF_P, (const uint8_t*)p.pcol + r0 * S::PW, R * S::PW, fb, pol);
        if constexpr (S::K0W > 0) bulk_g2s(d + B::OFF_K0, (const uint8_t*)p.k0 + r0 * S::K0W, R * S::K0W, fb, pol);
        if constexpr (S::K1W > 0) bulk_g2s(d + B::OFF_K1, (const uint8_t*)p.k1 + r0 * S::K1W, R * S::K1W, fb, pol);
#pragma unroll
        for (int i = 0; i < S::NC; ++i)
          bulk_g2s(d + B::OFF_C + i * R * 8, (const uint8_t*)p.col[i] + r0 * 8, R * 8, fb, pol);
        if (++stage == NS) {
          stage = 0;
          phase ^= 1;
        }
      }
    }
  } else {
    // ---- consumers
    KeyT<S> rk[L];
#pragma unroll
    for (int s = 0; s < L; ++s) rk[s] = (KeyT<S>)~0ULL;
    int stage = 0;
    uint32_t phase = 0;
    for (int64_t c = blockIdx.x; c < nfull; c += gridDim.x) {
      mbar_wait(&full[stage], phase);
      const uint8_t* d = stg + (size_t)stage * B::BYTES;
      uint64_t pr[UPW][2], k0[UPW][2], k1[UPW][2], cv[UPW][2][S::NC];
#pragma unroll
      for (int u = 0; u < UPW; ++u) {
        const int j = (wid * UPW + u) * 64 + 2 * lane;
        if constexpr (S::PW > 0) lds2<S::PW>(d + B::OFF_P, j, pr[u][0], pr[u][1]);
        if constexpr (S::K0W > 0) lds2<S::K0W>(d + B::OFF_K0, j, k0[u][0], k0[u][1]);
        if constexpr (S::K1W > 0) lds2<S::K1W>(d + B::OFF_K1, j, k1[u][0], k1[u][1]);
#pragma unroll
        for (int i = 0; i < S::NC; ++i) lds2<8>(d + B::OFF_C + i * R * 8, j, cv[u][0][i], cv[u][1][i]);
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
        priv_rows<S, L, T>(p, dir, rk, sm, tid, x[0], x[1], r);
      }
    }
    // ragged tail (< R rows): one CTA, scalar loads straight from global memory
    if (blockIdx.x == (int)(nfull % gridDim.x)) {
      for (int64_t base = nfull * R + (int64_t)wid * 64; base < n; base += 64 * NW) {
        const int64_t r = base + 2 * lane;
        SRow<S> x0, x1;
        spec_row_scalar<S>(p, r, x0);
        spec_row_scalar<S>(p, r + 1, x1);
        if (p.g.bitmap_out) emit_bitmap_unit(p.g, base, lane, x0.q, x1.q);
        priv_rows<S, L, T>(p, dir, rk, sm, tid, x0, x1, r);
      }
    }
  }
  priv_flush<S, L, T>(p, sm, dir, tid);
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
        priv_rows<S, L>(p, dir, rk, sm, tid, x[0], x[1], r);
      }
    } else {
      for (int u = 0; u < U; ++u) {
        const int64_t r = base + 64 * u + 2 * lane;
        SRow<S> x0, x1;
        spec_row_scalar<S>(p, r, x0);
        spec_row_scalar<S>(p, r + 1, x1);
        if (p.g.bitmap_out) emit_bitmap_unit(p.g, base + 64 * u, lane, x0.q, x1.q);
        priv_rows<S, L>(p, dir, rk, sm, tid, x0, x1, r);
      }
    }
  }
  priv_flush<S, L, T>(p, sm, dir, tid);
}

// ------------------------------------------------------------------ signature table
// TPC-H Q1 shape: pred i32; keys u8, u8; 4 decimal columns (qty, price, disc, tax);
// values: qty, price, price*(S-disc), price*(S-disc)*(S+tax), disc.
using SigQ1I = Sig<4, false, 1, 1, 4, false, vop(VX_COL, 0), vop(VX_COL, 1), vop(VX_M1, 1, 2), vop(VX_M1P, 1, 2, 3),
                   vop(VX_COL, 2)>;
using SigQ1F = Sig<4, false, 1, 1, 4, true, vop(VX_COL, 0), vop(VX_COL, 1), vop(VX_M1, 1, 2), vop(VX_M1P, 1, 2, 3),
                   vop(VX_COL, 2)>;

template <class S>
static bool spec_match(const Plan& g, SpecPlan* sp) {
  if (g.has_minmax) return false;
  if ((S::PW > 0) != (g.npreds == 1) || g.npreds > 1) return false;
  if (S::PW > 0 && (g.preds[0].col.width != S::PW || (bool)g.preds[0].is_f64 != S::PF64)) return false;
  if (g.nkeys != (S::K0W > 0) + (S::K1W > 0)) return false;
  if (S::K0W > 0 && g.keys[0].col.width != S::K0W) return false;
  if (S::K1W > 0 && g.keys[1].col.width != S::K1W) return false;
  if (g.nvals != S::NV) return false;
  // distinct operand columns in first-appearance order (a, b, c of each value)
  const void* cols[8];
  int32_t dts[8];
  int nc = 0;
  auto idx = [&](const DevCol& c) -> int {
    for (int i = 0; i < nc; ++i)
      if (cols[i] == c.ptr && dts[i] == c.dtype) return i;
    if (nc == 8) return 7;
    cols[nc] = c.ptr;
    dts[nc] = c.dtype;
    return nc++;
  };
  for (int v = 0; v < g.nvals; ++v) {
    const DevValue& d = g.vals[v];
    uint32_t op = S::OP(v);
    if ((int)vx_kind(op) != d.expr || (bool)d.is_f64 != S::F64 || d.off_sum < 0) return false;
    if (idx(d.a) != (int)vx_a(op)) return false;
    if (d.expr >= OCL_EXPR_MUL_1MINUS && idx(d.b) != (int)vx_b(op)) return false;
    if (d.expr >= OCL_EXPR_MUL_1MINUS_1PLUS && idx(d.c) != (int)vx_c(op)) return false;
  }
  if (nc != S::NC) return false;
  for (int i = 0; i < nc; ++i)
    if (dts[i] != (S::F64 ? OCL_F64 : OCL_I64)) return false;
  if (!g.vec_ok) return false;
  sp->g = g;
  sp->pcol = S::PW > 0 ? g.preds[0].col.ptr : nullptr;
  if (S::PW > 0 && S::PW < 8 && !S::PF64) {
    int64_t lo = g.preds[0].lo, hi = g.preds[0].hi;
    if (lo > hi || lo > INT32_MAX || hi < INT32_MIN) { sp->plo = 1; sp->phi = 0; }   // empty range
    else { sp->plo = (int32_t)(lo < INT32_MIN ? INT32_MIN : lo); sp->phi = (int32_t)(hi > INT32_MAX ? INT32_MAX : hi); }
  }
  sp->k0 = S::K0W > 0 ? g.keys[0].col.ptr : nullptr;
  sp->k1 = S::K1W > 0 ? g.keys[1].col.ptr : nullptr;
  for (int i = 0; i < 4; ++i) sp->col[i] = i < nc ? cols[i] : nullptr;
  return true;
}

template <class S>
static int spec_blocks_per_sm(size_t smem) {
  int nb = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&nb, k_sga_priv<S, kPrivSlots>, kPrivThreads, smem) != cudaSuccess ||
      nb < 1)
    nb = 1;
  return nb;
}

// Launch the bulk-pipeline kernel <S, L, T, R, NS>; false if it cannot run this plan
// (columns not 16-byte aligned for the copy engine, or fewer rows than one stage).
template <class S, int T, int R, int NS>
static bool launch_bulk(const SpecPlan& sp, int sms, cudaStream_t s, cudaError_t* err) {
  constexpr int L = kPrivSlots;
  auto a16 = [](const void* q) { return ((uintptr_t)q & 15) == 0; };
  if (sp.g.n < R) return false;
  if (S::PW > 0 && !a16(sp.pcol)) return false;
  if (S::K0W > 0 && !a16(sp.k0)) return false;
  if (S::K1W > 0 && !a16(sp.k1)) return false;
  for (int i = 0; i < S::NC; ++i)
    if (!a16(sp.col[i])) return false;
  auto fn = k_sga_bulk<S, L, T, R, NS>;
  const size_t smem = bulk_acc_bytes<S>(L, T) + (size_t)NS * BulkStage<S, R>::BYTES;
  static DevCache cache;
  const int nb = cache.get([&]() -> int {
    if (cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem) != cudaSuccess) return 0;
    int b = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, fn, T + 32, smem) != cudaSuccess || b < 1) b = 0;
    return b;
  });
  if (nb < 1) return false;
  int64_t grid = (int64_t)sms * nb;
  const int64_t chunks = sp.g.n / R;
  if (chunks < grid) grid = chunks;
  count_launch();
  fn<<<(int)grid, T + 32, smem, s>>>(sp);
  *err = cudaGetLastError();
  return true;
}

// Pipeline configuration, OCL_BULK = 0: off (the register-load kernel k_sga_priv);
// else <consumer threads, rows per stage, stages>: 1 = <256, 1024, 4>, 2 = <256, 512, 3>,
// 3 = <256, 512, 2>, 4 = <256, 512, 1>, 5 = <128, 256, 2>, 6 = <128, 256, 3>,
// 7 = <128, 512, 2>.  Default (OCL_BULK unset): 7 for int64 plans (3 CTAs x 4 consumer
// warps per SM; measured on B200 C4, profiles/r01_c4_bulk_configs.md), 3 for fp64 plans
// (C2: 51.0 -> 48.9 us, two sweeps agree, profiles/r01_c2_bulk_configs.md).
static int bulk_config() {
  const char* e = getenv("OCL_BULK");   // read per launch (tests switch it inside one process)
  return e ? atoi(e) : -1;
}

template <class S>
static bool launch_bulk_cfg(const SpecPlan& sp, int sms, cudaStream_t s, cudaError_t* err) {
  int cfg = bulk_config();
  if (cfg < 0) cfg = S::F64 ? 3 : 7;
  switch (cfg) {
    case 1: return launch_bulk<S, 256, 1024, 4>(sp, sms, s, err);
    case 2: return launch_bulk<S, 256, 512, 3>(sp, sms, s, err);
    case 3: return launch_bulk<S, 256, 512, 2>(sp, sms, s, err);
    case 4: return launch_bulk<S, 256, 512, 1>(sp, sms, s, err);
    case 5: return launch_bulk<S, 128, 256, 2>(sp, sms, s, err);
    case 6: return launch_bulk<S, 128, 256, 3>(sp, sms, s, err);
    case 7: return launch_bulk<S, 128, 512, 2>(sp, sms, s, err);
    default: return false;
  }
}

// Try the specialised low-G kernels; returns false if no signature matches.
// *kind: 1/2 = k_sga_priv (int / fp64), 3/4 = k_sga_bulk (int / fp64).
bool launch_fused_spec(const Plan& g, int sms, cudaStream_t s, cudaError_t* err, int* kind) {
  SpecPlan sp;
  int64_t tiles = (g.n + 127) / 128;
  auto go = [&](auto sig) -> bool {
    using S = decltype(sig);
    if (launch_bulk_cfg<S>(sp, sms, s, err)) {
      *kind += 2;
      return true;
    }
    const size_t smem = Acc<S>::bytes(kPrivSlots, kPrivThreads);
    static DevCache cache;
    const int nb = cache.get([&]() -> int {
      cudaFuncSetAttribute(k_sga_priv<S, kPrivSlots>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
      return spec_blocks_per_sm<S>(smem);
    });
    int grid = sms * nb;
    int64_t need = (tiles + 7) / 8;
    if (need < grid) grid = (int)(need > 0 ? need : 1);
    count_launch();
    k_sga_priv<S, kPrivSlots><<<grid, kPrivThreads, smem, s>>>(sp);
    *err = cudaGetLastError();
    return true;
  };
  if (spec_match<SigQ1I>(g, &sp)) { *kind = 1; return go(SigQ1I{}); }
  if (spec_match<SigQ1F>(g, &sp)) { *kind = 2; return go(SigQ1F{}); }
  return false;
}

}  // namespace ocl
