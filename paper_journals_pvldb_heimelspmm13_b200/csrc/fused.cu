// fused.cu — K9: fused select -> hash group -> aggregate, one pass over the columns.
//
// Paper steps fused here: selection (§4.1.1), hash group-by with
// dense group ids (L551-561 §4.1.6; hashing L511-533 §4.1.4), multi-column grouping
// on combined ids (L559-561), hierarchical grouped aggregation with per-work-group
// tables and several accumulators per group for few groups (L562-600 §4.1.7).
// Nothing is materialised: no bitmap (unless requested for tests), no oid list, no
// gid column.
//
// B200 design:
//  * Persistent grid (#SMs x resident CTAs).  A warp owns tiles of 128 rows; lane l
//    holds rows (2l, 2l+1) of each 64-row unit, so every column is read with one
//    vector load per lane per unit (u8 2 B, i32 8 B, i64/f64 16 B) and every
//    warp-wide load is one contiguous, fully used run (the paper's GPU pattern,
//    P:L619-633).
//  * Three places a qualifying row can be accumulated, tried in order:
//    1. PRIVATE slots: each thread owns one accumulator record per group slot in
//       shared memory ([slot][field][thread]); a CTA-wide directory maps the first 4
//       distinct keys to slots.  A row costs one slot-indexed read-modify-write per
//       accumulator: no atomics — the limit of the paper's "multiple accumulators
//       per group".  Few-group queries (TPC-H Q1) live entirely here;
//       with skewed keys the hot keys land here.
//    2. CTA TABLE (mid G): a shared-memory hash table with native 32-bit atomics
//       (sm_100 lowers 64-bit shared atomics to CAS loops): int32 values as 16-bit
//       split sums, flushed to HBM every 2^16 rows.
//    3. HBM TABLE: rows that miss are grouped per warp by key (__match_any_sync); one
//       leader per distinct key applies the group's combined update with global
//       atomics (int128 sums as two 64-bit atomics with carry from the returned value).
//    Rows whose values need int128 (int32-overflowing factors), or the key ~0, take an
//    exact per-row path.  Every path is exact; the tiers only decide speed.
//  * The kernel is templated on a *shape*: DynShape reads the plan's column widths and
//    expressions at run time (any plan); StaticShape<...> fixes them at compile time
//    (no dtype dispatch, every value column loaded once, narrow keys in 32 bits) — the
//    B200 stand-in for Ocelot's run-time kernel compilation.
//    Plans whose shape matches an instantiated StaticShape run the specialised code.
#include <stdlib.h>

#include "sga_device.cuh"

namespace ocl {

// ------------------------------------------------------------------ the kernel
template <class Sh, int NV, bool F64, bool MISS>
__global__ void __launch_bounds__(kFusedThreads) k_sga(const __grid_constant__ Plan p) {
  using Key = typename Sh::Key;
  constexpr int L = kRegSlots;
  constexpr int T = kFusedThreads;
  extern __shared__ __align__(16) uint8_t sm[];
  __shared__ uint64_t dir[L];
  __shared__ __align__(16) uint64_t blk[L * 32];   // CTA-level entry per slot (stride <= 256 B)
  __shared__ MissStage<MISS ? NV : 1, F64> stages[MISS ? T / 32 : 1];
  const int tid = threadIdx.x, lane = tid & 31;
  uint8_t* cta_tab = sm + (size_t)L * p.priv_rec * T;
  {
    uint4* z = (uint4*)sm;
    const int n16 = (int)(((size_t)L * p.priv_rec * T + (size_t)p.smem_cap * p.cta_stride) / 16);
    for (int i = tid; i < n16; i += T) z[i] = make_uint4(0, 0, 0, 0);
  }
  for (int i = tid; i < L * 32; i += T) blk[i] = 0;
  if (tid < L) dir[tid] = 0;
  __syncthreads();
  Key rk[L];
#pragma unroll
  for (int s = 0; s < L; ++s) rk[s] = (Key)~0ULL;   // never matches an admissible key
  MissStage<MISS ? NV : 1, F64>& stage = stages[MISS ? tid >> 5 : 0];

  const int64_t warp = (blockIdx.x * (int64_t)T + tid) >> 5;
  const int64_t nwarps = ((int64_t)gridDim.x * T) >> 5;
  if constexpr (Sh::kStatic && OCL_VAR_PIPE) {
    // Static shapes: 64-row units with a one-unit-ahead software pipeline — the next
    // unit's loads are in flight while the current unit is evaluated and placed.
    const int64_t nunits = (p.n + 63) / 64;
    const int64_t first = (int64_t)blockIdx.x * (T / 32);
    const int64_t rounds = nunits > first ? (nunits - first + nwarps - 1) / nwarps : 0;
    auto full = [&](int64_t u) { return p.vec_ok && u < nunits && u * 64 + 64 <= p.n; };
    RawUnit<Sh> cur, nxt;
    int64_t t = warp;
    if (full(t)) load_unit<Sh>(p, t * 64 + 2 * lane, cur);
    for (int64_t round = 0; round < rounds; ++round) {
      if (Sh::kCta && p.smem_cap && round > 0 && round % (kCtaFlushRounds * kUnits) == 0) {
        __syncthreads();
        for (int i = tid; i < p.smem_cap; i += T) cta_flush_entry(p, cta_tab + (size_t)i * p.cta_stride);
        __syncthreads();
      }
      const int64_t tn = t + nwarps;
      if (full(tn)) load_unit<Sh>(p, tn * 64 + 2 * lane, nxt);
      if (t < nunits) {
        const int64_t r = t * 64 + 2 * lane;
        Row<Sh, NV, F64> x0, x1;
        if (full(t)) {
          eval_unit<Sh, NV, F64>(p, cur, 0, x0);
          eval_unit<Sh, NV, F64>(p, cur, 1, x1);
        } else {
          eval_one<Sh, NV, F64>(p, r, x0);
          eval_one<Sh, NV, F64>(p, r + 1, x1);
        }
        if (p.bitmap_out) emit_bitmap_unit(p, t * 64, lane, x0.q, x1.q);
        place_row<Sh, NV, F64, MISS>(p, dir, rk, sm, cta_tab, tid, stage, x0, r);
        place_row<Sh, NV, F64, MISS>(p, dir, rk, sm, cta_tab, tid, stage, x1, r + 1);
      }
      cur = nxt;
      t = tn;
    }
  } else {
  const int64_t ntiles = (p.n + kTileRows - 1) / kTileRows;
  // CTA-uniform round count (the CTA's first warp has the most tiles): the whole CTA
  // meets at the periodic CTA-table flushes
  const int64_t first = (int64_t)blockIdx.x * (T / 32);
  const int64_t rounds = ntiles > first ? (ntiles - first + nwarps - 1) / nwarps : 0;
  for (int64_t round = 0; round < rounds; ++round) {
    if (Sh::kCta && p.smem_cap && round > 0 && round % kCtaFlushRounds == 0) {
      __syncthreads();
      for (int i = tid; i < p.smem_cap; i += T) cta_flush_entry(p, cta_tab + (size_t)i * p.cta_stride);
      __syncthreads();
    }
    const int64_t t = warp + round * nwarps;
    if (t >= ntiles) continue;
    const int64_t base = t * kTileRows;
    if (p.vec_ok && base + kTileRows <= p.n) {
      if constexpr (Sh::kStatic) {
        RawUnit<Sh> raw[kUnits];
#pragma unroll
        for (int u = 0; u < kUnits; ++u) load_unit<Sh>(p, base + 64 * u + 2 * lane, raw[u]);
#pragma unroll
        for (int u = 0; u < kUnits; ++u) {
          const int64_t r = base + 64 * u + 2 * lane;
          Row<Sh, NV, F64> x0, x1;
          eval_unit<Sh, NV, F64>(p, raw[u], 0, x0);
          eval_unit<Sh, NV, F64>(p, raw[u], 1, x1);
          if (p.bitmap_out) emit_bitmap_unit(p, base + 64 * u, lane, x0.q, x1.q);
          place_row<Sh, NV, F64, MISS>(p, dir, rk, sm, cta_tab, tid, stage, x0, r);
          place_row<Sh, NV, F64, MISS>(p, dir, rk, sm, cta_tab, tid, stage, x1, r + 1);
        }
      } else {
        Row<Sh, NV, F64> x[kUnits][2];
#pragma unroll
        for (int u = 0; u < kUnits; ++u) eval_pair<Sh, NV, F64>(p, base + 64 * u + 2 * lane, x[u][0], x[u][1]);
#pragma unroll
        for (int u = 0; u < kUnits; ++u) {
          const int64_t r = base + 64 * u + 2 * lane;
          if (p.bitmap_out) emit_bitmap_unit(p, base + 64 * u, lane, x[u][0].q, x[u][1].q);
          place_row<Sh, NV, F64, MISS>(p, dir, rk, sm, cta_tab, tid, stage, x[u][0], r);
          place_row<Sh, NV, F64, MISS>(p, dir, rk, sm, cta_tab, tid, stage, x[u][1], r + 1);
        }
      }
    } else {
      for (int u = 0; u < kUnits; ++u) {
        const int64_t r = base + 64 * u + 2 * lane;
        Row<Sh, NV, F64> x0, x1;
        eval_one<Sh, NV, F64>(p, r, x0);
        eval_one<Sh, NV, F64>(p, r + 1, x1);
        if (p.bitmap_out) emit_bitmap_unit(p, base + 64 * u, lane, x0.q, x1.q);
        place_row<Sh, NV, F64, MISS>(p, dir, rk, sm, cta_tab, tid, stage, x0, r);
        place_row<Sh, NV, F64, MISS>(p, dir, rk, sm, cta_tab, tid, stage, x1, r + 1);
      }
    }
  }

  }  // dynamic shapes

  // ---- flush: warp-reduce the private records -> CTA entry per slot -> HBM table
  __syncthreads();
  uint8_t* blkb = (uint8_t*)blk;
  for (int s = 0; s < L; ++s) {
    if (dir[s] == 0) continue;                       // uniform: slot never used in this CTA
    priv_flush_warp(p, sm + (size_t)s * p.priv_rec * T, tid, blkb + s * 256);
  }
  __syncthreads();
  if (tid < L) {
    const uint64_t sk = dir[tid];
    if (sk != 0) {
      uint8_t* e = table_find_or_insert(p.table, p.mask, p.stride, ~sk, p.status);
      if (e) entry_merge(p, blkb + tid * 256, e);
    }
  }
  if (Sh::kCta && p.smem_cap)
    for (int i = tid; i < p.smem_cap; i += T) cta_flush_entry(p, cta_tab + (size_t)i * p.cta_stride);
}

// ------------------------------------------------------------------ HBM-only tier (tier 2)
// Lanes own consecutive rows; runs of equal keys are folded by a segmented shuffle
// reduction into their first lane, which alone touches the table.
template <int NV, bool F64>
__global__ void __launch_bounds__(kFusedThreads) k_sga_glb(const __grid_constant__ Plan p) {
  using Sh = DynShape;
  const int lane = threadIdx.x & 31;
  const int64_t warp = (blockIdx.x * (int64_t)blockDim.x + threadIdx.x) >> 5;
  const int64_t nwarps = ((int64_t)gridDim.x * blockDim.x) >> 5;
  const int64_t nunits = (p.n + 31) / 32;
  for (int64_t t = warp; t < nunits; t += nwarps) {
    const int64_t r = t * 32 + lane;
    Row<Sh, NV, F64> x;
    eval_one<Sh, NV, F64>(p, r, x);
    if (p.bitmap_out) {
      const uint32_t w = __ballot_sync(0xffffffffu, x.q);
      if (lane == 0) p.bitmap_out[t] = w;
    }
    const bool ok = x.q && x.fast && x.key != ~0ULL;
    const unsigned okmask = __ballot_sync(0xffffffffu, ok);
    const uint64_t kprev = __shfl_up_sync(0xffffffffu, x.key, 1);
    const bool cont = ok && lane > 0 && ((okmask >> (lane - 1)) & 1u) && kprev == x.key;
    const unsigned contmask = __ballot_sync(0xffffffffu, cont);
    if (x.q && !ok) {                      // exact per-row path
      uint8_t* e = table_find_or_insert(p.table, p.mask, p.stride, x.key, p.status);
      if (e) update_entry_slow(p, e, r);
    }
    const unsigned later = lane == 31 ? 0u : (~contmask & ~((2u << lane) - 1u));
    const int seg_end = later ? __ffs(later) - 2 : 31;
    uint32_t c = ok ? 1u : 0u;
    I128 si[F64 ? 1 : NV];
    double sd[F64 ? NV : 1], mnd[F64 ? NV : 1], mxd[F64 ? NV : 1];
    int64_t mni[F64 ? 1 : NV], mxi[F64 ? 1 : NV];
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      if constexpr (F64) {
        sd[v] = ok ? x.vd[v] : 0.0;
        mnd[v] = mxd[v] = x.vd[v];
      } else {
        si[v] = ok ? i128_from_i64(x.vi[v]) : I128{0, 0};
        mni[v] = mxi[v] = x.vi[v];
      }
    }
    if (contmask) {
#pragma unroll
      for (int o = 1; o < 32; o <<= 1) {
        const bool take = lane + o <= seg_end;
        const uint32_t cy = __shfl_down_sync(0xffffffffu, c, o);   // every lane shuffles; `take` selects
        if (take) c += cy;
#pragma unroll
        for (int v = 0; v < NV; ++v) {
          if (v >= p.nvals) break;
          if constexpr (F64) {
            const double y = __shfl_down_sync(0xffffffffu, sd[v], o);
            const double a = __shfl_down_sync(0xffffffffu, mnd[v], o);
            const double b = __shfl_down_sync(0xffffffffu, mxd[v], o);
            if (take) {
              sd[v] += y;
              mnd[v] = fmin(mnd[v], a);
              mxd[v] = fmax(mxd[v], b);
            }
          } else {
            I128 y;
            y.lo = __shfl_down_sync(0xffffffffu, si[v].lo, o);
            y.hi = __shfl_down_sync(0xffffffffu, si[v].hi, o);
            const int64_t a = (int64_t)__shfl_down_sync(0xffffffffu, (long long)mni[v], o);
            const int64_t b = (int64_t)__shfl_down_sync(0xffffffffu, (long long)mxi[v], o);
            if (take) {
              si[v] = i128_add(si[v], y);
              mni[v] = min(mni[v], a);
              mxi[v] = max(mxi[v], b);
            }
          }
        }
      }
    }
    if (!ok || cont) continue;             // run heads only
    uint8_t* e = table_find_or_insert(p.table, p.mask, p.stride, x.key, p.status);
    if (!e) continue;
    atomicAdd((unsigned long long*)(e + 8), (unsigned long long)c);
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      if (v >= p.nvals) break;
      const DevValue& d = p.vals[v];
      if constexpr (F64) {
        if (d.off_sum >= 0) atomicAdd((double*)(e + d.off_sum), sd[v]);
        if (d.off_min >= 0) atomicMax((unsigned long long*)(e + d.off_min), (unsigned long long)enc_min_f(mnd[v]));
        if (d.off_max >= 0) atomicMax((unsigned long long*)(e + d.off_max), (unsigned long long)enc_max_f(mxd[v]));
      } else {
        if (d.is_f64) continue;
        if (d.off_sum >= 0) atomic_add_i128((uint64_t*)(e + d.off_sum), si[v].lo, si[v].hi);
        if (d.off_min >= 0) atomicMax((unsigned long long*)(e + d.off_min), (unsigned long long)enc_min_i(mni[v]));
        if (d.off_max >= 0) atomicMax((unsigned long long*)(e + d.off_max), (unsigned long long)enc_max_i(mxi[v]));
      }
    }
  }
}

// ------------------------------------------------------------------ static shapes (AOT instantiations)
// TPC-H Q1: pred i32; keys u8, u8; columns qty, price, disc, tax;
// values qty, price, price*(S-disc), price*(S-disc)*(S+tax), disc (SUMs).
using ShQ1I = StaticShape<4, false, 1, 1, 4, false, vop(0, VF_SUM, 0), vop(0, VF_SUM, 1), vop(1, VF_SUM, 1, 2),
                          vop(2, VF_SUM, 1, 2, 3), vop(0, VF_SUM, 2)>;
using ShQ1F = StaticShape<4, false, 1, 1, 4, true, vop(0, VF_SUM, 0), vop(0, VF_SUM, 1), vop(1, VF_SUM, 1, 2),
                          vop(2, VF_SUM, 1, 2, 3), vop(0, VF_SUM, 2)>;
// ------------------------------------------------------------------ dispatch
static size_t reg_smem(const Plan& p) {
  return (size_t)kRegSlots * p.priv_rec * kFusedThreads + (size_t)p.smem_cap * p.cta_stride;
}

template <class Sh, int NV, bool F64, bool MISS>
static cudaError_t launch_km(const Plan& p, int sms, cudaStream_t s) {
  const size_t smem = reg_smem(p);
  auto fn = k_sga<Sh, NV, F64, MISS>;
  cudaError_t e = cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  if (e != cudaSuccess) return e;
  int nb = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&nb, fn, kFusedThreads, smem) != cudaSuccess || nb < 1) nb = 1;
  int64_t grid = (int64_t)sms * nb;
  const int64_t need = ((p.n + kTileRows - 1) / kTileRows + (kFusedThreads / 32) - 1) / (kFusedThreads / 32);
  if (need < grid) grid = need > 0 ? need : 1;
  count_launch();
  fn<<<(int)grid, kFusedThreads, smem, s>>>(p);
  return cudaGetLastError();
}

// The warp-aggregated miss path is compiled in only for plans that expect more groups
// than private slots (Plan::miss_agg): few-group plans keep the lean row loop.
template <class Sh, int NV, bool F64>
static cudaError_t launch_k(const Plan& p, int sms, cudaStream_t s) {
  return p.miss_agg ? launch_km<Sh, NV, F64, true>(p, sms, s) : launch_km<Sh, NV, F64, false>(p, sms, s);
}

template <bool F64>
static cudaError_t launch_dyn(const Plan& p, int sms, cudaStream_t s) {
  if (p.nvals <= 1) return launch_k<DynShape, 1, F64>(p, sms, s);
  if (p.nvals <= 2) return launch_k<DynShape, 2, F64>(p, sms, s);
  if (p.nvals <= 4) return launch_k<DynShape, 4, F64>(p, sms, s);
  return launch_k<DynShape, 6, F64>(p, sms, s);
}

template <bool F64>
static cudaError_t launch_glb(const Plan& p, int sms, cudaStream_t s) {
  int64_t grid = (int64_t)sms * 8;
  const int64_t need = ((p.n + 31) / 32 + 7) / 8;
  if (need < grid) grid = need > 0 ? need : 1;
  count_launch();
  if (p.nvals <= 1) k_sga_glb<1, F64><<<(int)grid, kFusedThreads, 0, s>>>(p);
  else if (p.nvals <= 2) k_sga_glb<2, F64><<<(int)grid, kFusedThreads, 0, s>>>(p);
  else if (p.nvals <= 4) k_sga_glb<4, F64><<<(int)grid, kFusedThreads, 0, s>>>(p);
  else k_sga_glb<6, F64><<<(int)grid, kFusedThreads, 0, s>>>(p);
  return cudaGetLastError();
}

int reg_tier_slots() { return kRegSlots; }

// mode 0: plan-signature kernel if one matches, else the fused kernel (static shape if one
// matches); 1: fused kernel, DynShape only; 2: HBM-only kernel; 3: the fused kernel (no
// signature kernels: tier 4 forces its CTA shared-memory table).  values_f64: every value expression is fp64 (mixed plans use the
// integer instantiation, whose exact slow path handles fp64 values).  *kind reports
// the shape used (0 dynamic / HBM-only, 1.. static).
cudaError_t launch_fused(const Plan& p, int mode, bool values_f64, int sms, cudaStream_t s, int* kind) {
  *kind = 0;
  if (p.n == 0) return cudaSuccess;
  if (mode == 2) {
    *kind = 20;
    return values_f64 ? launch_glb<true>(p, sms, s) : launch_glb<false>(p, sms, s);
  }
  if (mode == 0 && p.vec_ok && getenv("OCL_NO_SPEC") == nullptr) {
    cudaError_t err = cudaSuccess;
    const bool aot = getenv("OCL_JIT_ALL") == nullptr;           // (A/B: every signature through NVRTC)
    if (aot && launch_fused_spec(p, sms, s, &err, kind)) return err;   // plan-signature kernels (fused_spec.cu)
    if (launch_fused_jit(p, sms, s, &err, kind)) return err;    // the same kernels compiled for this plan (jit.cu)
    *kind = 0;
  }
  if ((mode == 0 || mode == 3) && p.vec_ok) {
    if (shape_match<ShQ1I>(p)) {
      *kind = 1;
      return launch_k<ShQ1I, 5, false>(p, sms, s);
    }
    if (shape_match<ShQ1F>(p)) {
      *kind = 2;
      return launch_k<ShQ1F, 5, true>(p, sms, s);
    }
    if (shape_match<ShK64>(p)) {
      *kind = 3;
      return launch_k<ShK64, 1, false>(p, sms, s);
    }
    if (shape_match<ShP32K64>(p)) {
      *kind = 4;
      return launch_k<ShP32K64, 1, false>(p, sms, s);
    }
  }
  return values_f64 ? launch_dyn<true>(p, sms, s) : launch_dyn<false>(p, sms, s);
}

const char* fused_kernel_name(int kind) {
  switch (kind) {
    case 1: return "k_sga<StaticShape Q1 int64>";
    case 2: return "k_sga<StaticShape Q1 fp64>";
    case 3: return "k_sga<StaticShape key i64, COUNT/SUM/MIN/MAX>";
    case 4: return "k_sga<StaticShape pred i32, key i64, COUNT/SUM/MIN/MAX>";
    case 11: return "k_sga_priv<Sig Q1 int64>";
    case 12: return "k_sga_priv<Sig Q1 fp64>";
    case 13: return "k_sga_bulk<Sig Q1 int64> (TMA bulk pipeline)";
    case 14: return "k_sga_bulk<Sig Q1 fp64> (TMA bulk pipeline)";
    case 15: return "k_sga_bulk<Sig Q1+MINMAX int64> (TMA bulk pipeline)";
    case 16: return "k_sga_bulk<Sig Q1+MINMAX fp64> (TMA bulk pipeline)";
    case 61: return "k_sga_bulk<Sig pred i32, key i64, COUNT/SUM/MIN/MAX; 4 private slots>";
    case 64: return "k_sga_bulk<Sig pred i32, key i64, COUNT/SUM/MIN/MAX; CTA table>";
    case 71: return "k_sga_bulk<Sig key i64, COUNT/SUM/MIN/MAX; 4 private slots>";
    case 90: return "k_sga_bulk<Sig of the plan, run-time compiled (NVRTC); 4 private slots>";
    case 91: return "k_sga_bulk<Sig of the plan, run-time compiled (NVRTC); CTA table>";
    case 74: return "k_sga_bulk<Sig key i64, COUNT/SUM/MIN/MAX; CTA table>";
    case 20: return "k_sga_glb<DynShape>";
    case 30: return "k_part_count/scatter/agg<DynShape> (hash-partitioned)";
    case 31: return "k_part_count/scatter/agg<StaticShape key i64> (hash-partitioned)";
    case 32: return "k_part_count/scatter/agg<StaticShape pred i32, key i64> (hash-partitioned)";
    case 40: return "k_sorted_summary/scan/agg<DynShape> (sorted input)";
    case 41: return "k_sorted_summary/scan/agg<StaticShape key i64> (sorted input)";
    case 42: return "k_sorted_summary/scan/agg<StaticShape pred i32, key i64> (sorted input)";
    case 50: return "k_rs_* radix sort + k_sorted_*<DynShape> (tier 6)";
    case 51: return "k_rs_* radix sort + k_sorted_*<StaticShape key i64> (tier 6)";
    case 52: return "k_rs_* radix sort + k_sorted_*<StaticShape pred i32, key i64> (tier 6)";
    default: return "k_sga<DynShape>";
  }
}

}  // namespace ocl
