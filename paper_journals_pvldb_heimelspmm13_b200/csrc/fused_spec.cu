// fused_spec.cu — plan-signature fused kernels: select -> group -> aggregate in one
// pass over TMA-streamed columns, specialised at compile time for the plan shapes the
// benchmark configurations use (TPC-H Q1, Q1 + MIN/MAX, and the GROUP BY key / COUNT,
// SUM, MIN, MAX shape of C3 / C5).
//
// Same method, semantics and accumulation scheme as the unified kernel in fused.cu
// (§4.1.1 selection, §4.1.6 grouping, §4.1.7 aggregation), specialised by hand:
// compile-time column widths, key packing and accumulator layout.  The columns reach
// shared memory through the copy engine (k_sga_bulk: cp.async.bulk + an mbarrier ring
// fed by one producer warp) so the consumer warps only compute; k_sga_priv is the
// register-load variant for inputs smaller than one pipeline stage.
//
// Accumulation tiers (§4.1.7: local accumulation, "multiple accumulators per
// group, inversely proportional to the number of groups"), chosen by expected_groups:
//  * private (<= 4 groups): every consumer thread owns one accumulator record per group slot
//    in shared memory ([slot][field][thread]: lane t always hits the same banks); a row
//    costs a register compare against the 4 slot keys and a non-atomic read-modify-write —
//    the limit of the paper's accumulators ∝ 1/G.
//  * CTA table (<= 2048 groups, integer COL values): one shared-memory hash table per CTA,
//    as large as fits (tab_policy: replicas did not pay on B200), stored field-major, native
//    32-bit shared atomics — count, biased 64-bit sums as a 32-bit add whose carry is taken
//    from the returned value (exact, no periodic fold), order-encoded MIN / MAX — and
//    slot-granular linear probing (one LDS.64 for a home-slot hit).
// Rows outside the int32 fast path, the key ~0 and keys beyond the tier's capacity take
// the exact per-row update of the HBM table.  At the end every CTA folds its records /
// table into the HBM table (int128 sums).
//
// On B200, C4 (600M rows, Q1) runs in ~3.5 ms (~98-100 % of the measured copy bandwidth).
// launch_fused (fused.cu) tries these kernels first; OCL_NO_SPEC=1 disables them.
#include <stdio.h>

#include "launch.cuh"
#include "spec_device.cuh"

namespace ocl {

// ------------------------------------------------------------------ signature table
// TPC-H Q1 shape: pred i32; keys u8, u8; 4 decimal columns (qty, price, disc, tax);
// values: qty, price, price*(S-disc), price*(S-disc)*(S+tax), disc.
using SigQ1I = Sig<4, false, 1, 1, 4, false, vop(VX_COL, 0), vop(VX_COL, 1), vop(VX_M1, 1, 2), vop(VX_M1P, 1, 2, 3),
                   vop(VX_COL, 2)>;
using SigQ1F = Sig<4, false, 1, 1, 4, true, vop(VX_COL, 0), vop(VX_COL, 1), vop(VX_M1, 1, 2), vop(VX_M1P, 1, 2, 3),
                   vop(VX_COL, 2)>;
// Q1 + MIN(qty) + MAX(price) (bench workload c4mm): the same columns, two more states.
using SigQ1IMM = Sig<4, false, 1, 1, 4, false, vop(VX_COL, 0, 0, 0, VS_SUM | VS_MIN),
                     vop(VX_COL, 1, 0, 0, VS_SUM | VS_MAX), vop(VX_M1, 1, 2), vop(VX_M1P, 1, 2, 3), vop(VX_COL, 2)>;
using SigQ1FMM = Sig<4, false, 1, 1, 4, true, vop(VX_COL, 0, 0, 0, VS_SUM | VS_MIN),
                     vop(VX_COL, 1, 0, 0, VS_SUM | VS_MAX), vop(VX_M1, 1, 2), vop(VX_M1P, 1, 2, 3), vop(VX_COL, 2)>;
// C5: WHERE p (i32) GROUP BY key (i64): COUNT, SUM, MIN, MAX of v (i64).  C3: the same
// without the predicate (GROUP BY l_orderkey: COUNT, SUM / MIN / MAX(l_quantity)).
using SigC5 = Sig<4, false, 8, 0, 1, false, vop(VX_COL, 0, 0, 0, VS_SUM | VS_MIN | VS_MAX)>;
using SigC3 = Sig<0, false, 8, 0, 1, false, vop(VX_COL, 0, 0, 0, VS_SUM | VS_MIN | VS_MAX)>;

// Select-compact-gather threshold (k_sga_bulk): CTAs whose predicate sample selects less
// than this many percent of the rows stream the predicate column only and gather the
// qualifying rows' key / value sectors.  Off below 2^24 rows, where the sample's latency at
// kernel start is not amortised.  OCL_SPARSE_PCT overrides (0 = off).
int32_t spec_sparse_pct(int64_t n) {
  if (const char* e = getenv("OCL_SPARSE_PCT")) return atoi(e);
  return n >= ((int64_t)1 << 24) ? 8 : 0;
}

// The threshold a launch uses: 0 without a predicate; on the private tier (<= 4 groups) 0
// unless OCL_SPARSE_PCT is set — the twin's early exit costs its 3 x 148 CTAs ~16 us
// (C4 3.46 -> 3.49 ms), more than the mode is worth there (C5 G = 4 at 1 %: 0.86 -> 0.74 ms).
int32_t spec_twin_pct(int32_t pct, bool has_pred, bool private_tier) {
  if (!has_pred || (private_tier && !getenv("OCL_SPARSE_PCT"))) return 0;
  return pct;
}

template <class S>
static bool spec_match(const Plan& g, SpecPlan* sp) {
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
    if ((int)vx_kind(op) != d.expr || (bool)d.is_f64 != S::F64) return false;
    if ((d.off_sum >= 0) != S::has(v, VS_SUM) || (d.off_min >= 0) != S::has(v, VS_MIN) ||
        (d.off_max >= 0) != S::has(v, VS_MAX))
      return false;
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
  sp->tab_hb = 0;
  sp->tab_nrep = 0;
  sp->pwait = 0;
  sp->cwait = 0;
  sp->mm_check = 0;
  sp->sparse_pct = spec_sparse_pct(g.n);
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
template <class S, int L, int T, int R, int NS>
static bool launch_bulk(const SpecPlan& sp, int sms, cudaStream_t s, cudaError_t* err) {
  auto a16 = [](const void* q) { return ((uintptr_t)q & 15) == 0; };
  if (sp.g.n < R) return false;
  if (S::PW > 0 && !a16(sp.pcol)) return false;
  if (S::K0W > 0 && !a16(sp.k0)) return false;
  if (S::K1W > 0 && !a16(sp.k1)) return false;
  for (int i = 0; i < S::NC; ++i)
    if (!a16(sp.col[i])) return false;
  auto fn = k_sga_bulk<S, L, T, R, NS>;
  const size_t smem = tier_bytes<S, L>(T, sp.tab_nrep << sp.tab_hb) + (size_t)NS * BulkStage<S, R>::BYTES;
  // per device: the kernel's dynamic shared-memory attribute, raised to the largest size
  // launched so far (an attribute far above the need changed the SM's carveout choice and
  // cost ~15 % on C4); per device and table size: the resident CTAs per SM
  static DevCache attr;
  int have = attr.get([&]() -> int { return 0; });
  if ((int)smem > have) {
    if (cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem) != cudaSuccess) {
      cudaGetLastError();
      return false;
    }
    int d = 0;
    cudaGetDevice(&d);
    if (d >= 0 && d < kMaxDevices) attr.v[d].store((int)smem, std::memory_order_relaxed);
  }
  static DevCache cache[8];
  int ci = 0;
  for (uint32_t c = sp.tab_nrep << sp.tab_hb; c > 128 && ci < 7; c >>= 1) ++ci;
  const int nb = cache[ci].get([&]() -> int {
    int b = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, fn, T + 32, smem) != cudaSuccess || b < 1) {
      cudaGetLastError();
      b = 0;
    }
    return b;
  });
  if (nb < 1) return false;
  int64_t grid = (int64_t)sms * nb;
  const int64_t chunks = sp.g.n / R;
  if (chunks < grid) grid = chunks;
  SpecPlan q = sp;
  if (const char* w = getenv("OCL_WAIT")) {        // "<producer><consumer>" digits, e.g. "10"
    q.pwait = w[0] ? w[0] - '0' : 0;
    q.cwait = w[0] && w[1] ? w[1] - '0' : 0;
  }
  q.sparse_pct = spec_twin_pct(q.sparse_pct, S::PW > 0, L > 0);
  if (getenv("OCL_DEBUG"))
    fprintf(stderr, "[ocl] k_sga_bulk L=%d T=%d R=%d NS=%d tab=%u x 2^%u smem=%zu blocks/SM=%d grid=%lld sparse<%d%%\n",
            L, T, R, NS, q.tab_nrep, q.tab_hb, smem, nb, (long long)grid, q.sparse_pct);
  if constexpr (S::PW > 0) {
    // select-compact-gather twin first: exactly one of the two kernels runs past its sample
    if (q.sparse_pct > 0) {
      auto fs = k_sga_sparse<S, L, T, R, NS>;
      static DevCache sattr;
      if ((int)smem > sattr.get([&]() -> int { return 0; })) {
        if (cudaFuncSetAttribute(fs, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem) != cudaSuccess) {
          cudaGetLastError();
          return false;
        }
        int d = 0;
        cudaGetDevice(&d);
        if (d >= 0 && d < kMaxDevices) sattr.v[d].store((int)smem, std::memory_order_relaxed);
      }
      count_launch();
      fs<<<(int)grid, T + 32, smem, s>>>(q);
      if ((*err = cudaGetLastError()) != cudaSuccess) return true;
    }
  }
  count_launch();
  fn<<<(int)grid, T + 32, smem, s>>>(q);
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
static bool launch_bulk_cfg(const SpecPlan& sp, int sms, cudaStream_t s, cudaError_t* err, int dflt = -1) {
  int cfg = bulk_config();
  if (cfg < 0) cfg = dflt >= 0 ? dflt : (S::F64 ? 3 : 7);
  constexpr int L = kPrivSlots;
  switch (cfg) {
    case 1: return launch_bulk<S, L, 256, 1024, 4>(sp, sms, s, err);
    case 2: return launch_bulk<S, L, 256, 512, 3>(sp, sms, s, err);
    case 3: return launch_bulk<S, L, 256, 512, 2>(sp, sms, s, err);
    case 4: return launch_bulk<S, L, 256, 512, 1>(sp, sms, s, err);
    case 5: return launch_bulk<S, L, 128, 256, 2>(sp, sms, s, err);
    case 6: return launch_bulk<S, L, 128, 256, 3>(sp, sms, s, err);
    case 7: return launch_bulk<S, L, 128, 512, 2>(sp, sms, s, err);
    default: return false;
  }
}

// Few-group signatures (L = 4): the bulk pipeline (*kind + 2), else the register-load
// kernel (fewer rows than one stage, or OCL_BULK=0).
template <class S>
static bool launch_few(const SpecPlan& sp, int sms, cudaStream_t s, cudaError_t* err, int* kind) {
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
  const int64_t tiles = (sp.g.n + 127) / 128;
  const int64_t need = (tiles + 7) / 8;
  if (need < grid) grid = (int)(need > 0 ? need : 1);
  count_launch();
  k_sga_priv<S, kPrivSlots><<<grid, kPrivThreads, smem, s>>>(sp);
  *err = cudaGetLastError();
  return true;
}

// Group-by signatures: the tier by expected groups — 4 private slots, or one shared-memory
// hash table per CTA (<= kSpecTabMaxGroups groups).  false: no tier fits (the caller falls back).
constexpr int64_t kSpecTabMaxGroups = 2048;

// CTA table: read-before-atomic MIN / MAX (smem_max), on by default: +0-4 % on uniform keys,
// -25..45 % with Zipf 1.5 (C5 G = 16 1.89 -> 1.16 ms, G = 256 1.79 -> 1.26 ms, G = 2048
// 2.07 -> 1.52 ms).  OCL_MM_CHECK=0/1 forces it (A/B).
int32_t spec_mm_check(int64_t eg) {
  (void)eg;
  if (const char* e = getenv("OCL_MM_CHECK")) return atoi(e) != 0;
  return 1;
}

// CTA-table policy (shared with the run-time compiled kernels, jit.cu).  Measured on B200, C5
// on 2^28 rows (profiles/r02_tab_policy.md):
//  - one table per CTA, as large as fits: replicas per warp group (the paper's "multiple
//    accumulators") never paid here — across warps, shared atomics on one
//    address cost no more than on different ones, while every replica raises the load
//    factor of a fixed budget (G = 512: 2 replicas x 1024 slots 3.11 ms, 1 x 2048 1.80 ms);
//  - one CTA of 30 consumer warps per SM (<960, 1920, 2>) with a 4096-slot table beats two
//    CTAs of 16 warps with 2048 slots each at every G (G = 256 1.51 -> 1.26 ms);
//  - slot-granular probing (one LDS.64 per row) beat buckets of 4 slots (two LDS.128) at
//    every load up to 1/2 except G = 1024 uniform (1.52 vs 1.60 ms), so only slots remain.
// Rows wider than the 30-warp stages allow fall back to <512, 1024, 2> (run-time compiled
// signatures only).  The table must keep the load <= 1/2.  OCL_TAB="<wide|narrow>,<log2
// slots>,<tables>" overrides (A/B).
bool tab_policy(int64_t eg, size_t slot_bytes, size_t row_bytes, TabPolicy* tp) {
  constexpr size_t kSmem = 225 * 1024;            // per SM, minus the static / reserved bytes
  auto fit = [&](size_t budget) -> uint32_t {     // log2 of the largest table within budget
    uint32_t hb = 0;
    while (((size_t)2 << hb) * slot_bytes <= budget && hb < 16) ++hb;
    return hb;
  };
  *tp = TabPolicy{};
  tp->nrep = 1;
  tp->NS = 2;
  for (int wide = 1; wide >= 0 && tp->T == 0; --wide) {
    const int R = wide ? 1920 : 1024;
    const size_t stages = 2 * (size_t)R * row_bytes;
    if (stages >= kSmem) continue;
    const uint32_t hb = fit(kSmem - stages);
    if (hb >= 6 && ((int64_t)1 << hb) >= 2 * eg) tp->T = wide ? 960 : 512, tp->R = R, tp->hb = hb;
  }
  if (const char* e = getenv("OCL_TAB")) {
    char kind[8] = {0};
    int a = 0, b = 0;
    if (sscanf(e, "%6[a-z],%d,%d", kind, &a, &b) == 3 && a >= 6 && b >= 1) {
      const bool wide = kind[0] == 'w';
      const size_t stages = 2 * (size_t)(wide ? 1920 : 1024) * row_bytes;
      if (((size_t)b << a) * slot_bytes + stages <= kSmem)
        tp->T = wide ? 960 : 512, tp->R = wide ? 1920 : 1024, tp->hb = (uint32_t)a, tp->nrep = (uint32_t)b;
    }
  }
  if (tp->T == 0) return false;
  tp->mm_check = spec_mm_check(eg);
  return true;
}

template <class S>
static bool launch_grp(SpecPlan& sp, int sms, cudaStream_t s, cudaError_t* err, int* tier) {
  const int64_t eg = sp.g.expected > 0 ? sp.g.expected : 1;
  if (eg <= 4) { *tier = 1; return launch_bulk<S, 4, 128, 512, 2>(sp, sms, s, err); }
  if constexpr (S::cta_ok()) {
    TabPolicy tp;
    if (eg <= kSpecTabMaxGroups && tab_policy(eg, TabL<S>::BYTES_PER_SLOT, BulkStage<S, 64>::BYTES / 64, &tp) &&
        tp.T == 960) {                            // (the C5 / C3 rows always fit the wide stages)
      sp.tab_hb = tp.hb;
      sp.tab_nrep = tp.nrep;
      sp.mm_check = tp.mm_check;
      *tier = 4;
      return launch_bulk<S, 0, 960, 1920, 2>(sp, sms, s, err);
    }
  }
  return false;
}

// Whether a group-by signature kernel takes this plan (the planner then keeps the one-pass
// fused kernel instead of the hash-partitioned tier).
bool spec_takes(const Plan& g) {
  SpecPlan sp;
  const int64_t eg = g.expected > 0 ? g.expected : 1;
  if (eg > kSpecTabMaxGroups || getenv("OCL_NO_SPEC")) return false;
  return spec_match<SigC5>(g, &sp) || spec_match<SigC3>(g, &sp);
}

// Try the specialised kernels; returns false if no signature matches.  *kind (see
// fused_kernel_name): 11/12 = k_sga_priv Q1 (int / fp64), 13/14 = k_sga_bulk Q1, 15/16 =
// k_sga_bulk Q1 + MIN/MAX, 60 + tier = C5 shape, 70 + tier = C3 shape (tier 1 = 4 private
// slots, 4 = CTA table).
bool launch_fused_spec(const Plan& g, int sms, cudaStream_t s, cudaError_t* err, int* kind) {
  SpecPlan sp;
  const int64_t eg = g.expected > 0 ? g.expected : 1;
  if (eg <= kPrivSlots) {
    if (spec_match<SigQ1I>(g, &sp)) { *kind = 11; return launch_few<SigQ1I>(sp, sms, s, err, kind); }
    if (spec_match<SigQ1F>(g, &sp)) { *kind = 12; return launch_few<SigQ1F>(sp, sms, s, err, kind); }
    if (spec_match<SigQ1IMM>(g, &sp)) {
      *kind = 15;                           // <128, 256, 3>: 4.19 -> 4.07 ms on c4mm (vs <128, 512, 2>)
      return launch_bulk_cfg<SigQ1IMM>(sp, sms, s, err, 6);
    }
    if (spec_match<SigQ1FMM>(g, &sp)) {
      *kind = 16;
      return launch_bulk_cfg<SigQ1FMM>(sp, sms, s, err);
    }
  }
  int t = 0;
  if (spec_match<SigC5>(g, &sp) && launch_grp<SigC5>(sp, sms, s, err, &t)) { *kind = 60 + t; return true; }
  if (spec_match<SigC3>(g, &sp) && launch_grp<SigC3>(sp, sms, s, err, &t)) { *kind = 70 + t; return true; }
  return false;
}

}  // namespace ocl
