// aggregate.cu — K8: grouped aggregation over a dense group-id column (unfused chain).
//
// Paper (§4.1.7): work-groups on disjoint partitions build
// intermediate aggregation tables with atomics in local memory; for few groups each
// group is spread over several accumulators ("the number of accumulators per group
// being chosen inversely proportional to the number of groups") to cut same-address
// contention; tables that do not fit local memory fall back to the same scheme in
// global memory.  Then one thread per group finalises (k_finalize_dense).
//
// B200 design: the same three tiers as the fused kernel (sga_device.cuh), indexed by
// the group id instead of a hashed key:
//   PRIVATE  (G small): one accumulator record per group per thread in shared memory
//            ([g][field][thread]) — the paper's multiple accumulators taken to one per
//            thread: no atomics at all in the row loop;
//   CTA      (G fits shared memory, integer COL values): a direct-indexed array of
//            32-bit-field entries updated with native shared-memory atomics, flushed to
//            HBM every 2^16 rows;
//   HBM      otherwise: warp-aggregated (__match_any_sync on the gid) global atomics.
// Values are read at row oids[j] (a fused gather).  Rows whose values need int128 go
// through the exact per-row path.
#include <algorithm>

#include "sga_device.cuh"

namespace ocl {

constexpr size_t kAggSmemBudget = 160 * 1024;
#ifndef OCL_GAGG_R
#define OCL_GAGG_R 8
#endif

// Static shapes: the NC distinct value columns of row r were gathered into c[] by the
// caller (all loads of a thread's R rows are issued before any update).
template <class Sh, int NV, bool F64>
__device__ __forceinline__ void agg_eval(const Plan& p, int64_t r, int32_t g, const uint64_t* c,
                                         Row<Sh, NV, F64>& x) {
  x.q = true;
  x.fast = true;
  x.bad = 0;
  x.key = (typename Sh::Key)(uint32_t)g;
  if constexpr (Sh::kStatic) {
#pragma unroll
    for (int v = 0; v < NV; ++v) value_of<Sh, NV, F64>(p, v, c[Sh::ia(v)], c[Sh::ib(v)], c[Sh::ic(v)], x);
  } else {
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      if (v >= p.nvals) break;
      const DevValue& d = p.vals[v];
      if (!F64 && d.is_f64) {
        x.fast = false;
        continue;
      }
      const uint64_t a = ld1w(d.a.width, d.a.ptr, r);
      const uint64_t b = d.expr >= OCL_EXPR_MUL_1MINUS ? ld1w(d.b.width, d.b.ptr, r) : 0;
      const uint64_t cc = d.expr >= OCL_EXPR_MUL_1MINUS_1PLUS ? ld1w(d.c.width, d.c.ptr, r) : 0;
      value_of<Sh, NV, F64>(p, v, a, b, cc, x);
    }
  }
  x.fast = x.fast && x.bad == 0;
}

// Group g goes to the private records when g < npriv, else to the CTA array when
// g < ncta (integer COL values), else to the warp-aggregated HBM update.
template <class Sh, int NV, bool F64>
__global__ void __launch_bounds__(kFusedThreads) k_group_aggregate(const __grid_constant__ Plan p, int64_t max_rows,
                                                                   const int64_t* ngroups_dev, int64_t max_groups,
                                                                   int32_t npriv, int32_t ncta) {
  constexpr int T = kFusedThreads;
  extern __shared__ __align__(16) uint8_t sm[];
  __shared__ MissStage<NV, F64> stages[T / 32];
  const int tid = threadIdx.x;
  int64_t G = ngroups_dev ? *ngroups_dev : max_groups;
  if (G > max_groups) G = max_groups;
  const int64_t m = p.m_dev ? *p.m_dev : max_rows;
  const int64_t np_ = npriv < G ? npriv : G;
  const int64_t nc_ = ncta < G ? ncta : G;
  uint8_t* cta = sm + (size_t)npriv * p.priv_rec * T;
  {
    const size_t bytes = (size_t)np_ * p.priv_rec * T;
    uint4* z = (uint4*)sm;
    for (int64_t i = tid; i < (int64_t)(bytes / 16); i += T) z[i] = make_uint4(0, 0, 0, 0);
    uint4* zc = (uint4*)cta;
    for (int64_t i = tid; i < (int64_t)((size_t)nc_ * p.cta_stride / 16); i += T) zc[i] = make_uint4(0, 0, 0, 0);
    __syncthreads();
  }
  MissStage<NV, F64>& stage = stages[tid >> 5];
  // R rows per thread per round: every gid/oid/value load of the R rows is in flight
  // before the first update (the value loads depend on the oid loads: memory-level
  // parallelism, not bandwidth, bounds a one-row-at-a-time gather).
  // 8: 7.17 -> 6.49 ms on the Q1 set at 600M rows (16: 9.9).  Also measured (round 2, same box,
  // 6.48 ms base): R = 4 at 3 CTAs/SM 7.25, R = 4 / 2 at 4 CTAs/SM 8.28 / 8.84, R = 6 at 3 CTAs/SM
  // 8.14 (spills)
  constexpr int R = Sh::kStatic ? OCL_GAGG_R : 1;
  constexpr int NCc = Sh::kStatic ? Sh::NC : 1;
  constexpr int64_t kFlushRounds = 256 / R;                   // 2^16 rows per CTA between CTA-tier flushes
  const int64_t per_round = (int64_t)gridDim.x * T * R;
  const int64_t rounds = (m + per_round - 1) / per_round;    // uniform across the grid
  for (int64_t round = 0; round < rounds; ++round) {
    if (nc_ > np_ && round > 0 && round % kFlushRounds == 0) {
      __syncthreads();
      for (int64_t g = np_ + tid; g < nc_; g += T) cta_flush_entry(p, cta + g * p.cta_stride, g);
      __syncthreads();
    }
    const int64_t base = round * per_round + (int64_t)blockIdx.x * T * R + tid;
    int32_t gk[R];
    int64_t rk[R];
    uint64_t c[R][NCc];
#pragma unroll
    for (int k = 0; k < R; ++k) {
      const int64_t j = base + (int64_t)k * T;
      gk[k] = j < m ? __ldg(p.gids + j) : -1;
      rk[k] = j < m ? (p.oids ? (int64_t)__ldg(p.oids + j) : j) : -1;
    }
    // the oid and value loads do not wait for the gid (row j < m has a valid oid): two
    // dependent round trips (gid || oid -> values) instead of three (gid -> oid -> values):
    // Q1 set at 600M rows 6.48 -> 5.14 ms
    if constexpr (Sh::kStatic) {
#pragma unroll
      for (int k = 0; k < R; ++k)
#pragma unroll
        for (int i = 0; i < NCc; ++i)
          c[k][i] = rk[k] >= 0 ? (uint64_t)__ldg((const long long*)p.vcols[i].ptr + rk[k]) : 0;
    }
#pragma unroll
    for (int k = 0; k < R; ++k)
      if (gk[k] >= G) gk[k] = -1;
#pragma unroll
    for (int k = 0; k < R; ++k) {
      const int32_t g = gk[k];
      const int64_t r = rk[k];
      const bool valid = g >= 0;
      Row<Sh, NV, F64> x;
      if (valid) {
        agg_eval<Sh, NV, F64>(p, r, g, c[k], x);
      } else {
        x.q = false;
        x.fast = true;
        x.bad = 0;
        x.key = 0;
      }
      bool miss = false;
      if (valid) {
        if (!x.fast) update_entry_slow(p, p.table + (int64_t)g * p.stride, r);
        else if (g < np_) priv_add<Sh, NV, F64>(p, sm, g, tid, x);
        else if (g < nc_) cta_add<Sh, NV, F64>(p, cta + (int64_t)g * p.cta_stride, x);
        else miss = true;
      }
      warp_miss_update<Sh, NV, F64>(p, stage, miss, x, tid & 31);   // (always on: G may exceed the tiers)
    }
  }
  __syncthreads();
  for (int64_t g = 0; g < np_; ++g) priv_flush_warp(p, sm + (size_t)g * p.priv_rec * T, tid, p.table + g * p.stride);
  for (int64_t g = np_ + tid; g < nc_; g += T) cta_flush_entry(p, cta + g * p.cta_stride, g);
}

template <class Sh, int NV, bool F64>
static cudaError_t launch_agg_nv(const Plan& p, int64_t max_rows, const int64_t* ngroups_dev, int64_t max_groups,
                                 int sms, cudaStream_t s) {
  // private records for the first groups (up to 64 KB: three CTAs per SM), then a CTA
  // array for integer COL plans
  int64_t npriv = std::min<int64_t>(max_groups, (int64_t)(64 * 1024 / ((size_t)p.priv_rec * kFusedThreads)));
  bool int_cols = true;
  for (int v = 0; v < p.nvals; ++v) int_cols = int_cols && !p.vals[v].is_f64 && p.vals[v].expr == OCL_EXPR_COL;
  int64_t ncta = npriv;
  if (int_cols && !F64)
    ncta = std::min<int64_t>(max_groups, npriv + (int64_t)((kAggSmemBudget - (size_t)npriv * p.priv_rec * kFusedThreads) /
                                                            (size_t)p.cta_stride));
  const size_t smem = (size_t)npriv * p.priv_rec * kFusedThreads + (size_t)ncta * p.cta_stride;
  auto fn = k_group_aggregate<Sh, NV, F64>;
  cudaError_t e = cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
  if (e != cudaSuccess) return e;
  int nb = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&nb, fn, kFusedThreads, smem) != cudaSuccess || nb < 1) nb = 1;
  int64_t grid = (int64_t)sms * nb;
  const int64_t need = (max_rows + kFusedThreads * 4 - 1) / (kFusedThreads * 4);
  if (need < grid) grid = need > 0 ? need : 1;
  count_launch();
  fn<<<(int)grid, kFusedThreads, smem, s>>>(p, max_rows, ngroups_dev, max_groups, (int32_t)npriv, (int32_t)ncta);
  return cudaGetLastError();
}

// Static value shapes of the grouped aggregation: the TPC-H Q1 value set (int64 and
// fp64 decimals) and COUNT/SUM/MIN/MAX of one int64 column.
using AgQ1I = StaticShape<0, false, 0, 0, 4, false, vop(0, VF_SUM, 0), vop(0, VF_SUM, 1), vop(1, VF_SUM, 1, 2),
                          vop(2, VF_SUM, 1, 2, 3), vop(0, VF_SUM, 2)>;
using AgQ1F = StaticShape<0, false, 0, 0, 4, true, vop(0, VF_SUM, 0), vop(0, VF_SUM, 1), vop(1, VF_SUM, 1, 2),
                          vop(2, VF_SUM, 1, 2, 3), vop(0, VF_SUM, 2)>;
using AgV1 = StaticShape<0, false, 0, 0, 1, false, vop(0, VF_SUM | VF_MIN | VF_MAX, 0)>;

template <bool F64>
static cudaError_t launch_agg_f(const Plan& p, int64_t max_rows, const int64_t* ngroups_dev, int64_t max_groups,
                                int sms, cudaStream_t s) {
  if (!F64 && values_match<AgQ1I>(p)) return launch_agg_nv<AgQ1I, 5, false>(p, max_rows, ngroups_dev, max_groups, sms, s);
  if (F64 && values_match<AgQ1F>(p)) return launch_agg_nv<AgQ1F, 5, true>(p, max_rows, ngroups_dev, max_groups, sms, s);
  if (!F64 && values_match<AgV1>(p)) return launch_agg_nv<AgV1, 1, false>(p, max_rows, ngroups_dev, max_groups, sms, s);
  if (p.nvals <= 1) return launch_agg_nv<DynShape, 1, F64>(p, max_rows, ngroups_dev, max_groups, sms, s);
  if (p.nvals <= 2) return launch_agg_nv<DynShape, 2, F64>(p, max_rows, ngroups_dev, max_groups, sms, s);
  if (p.nvals <= 4) return launch_agg_nv<DynShape, 4, F64>(p, max_rows, ngroups_dev, max_groups, sms, s);
  return launch_agg_nv<DynShape, 6, F64>(p, max_rows, ngroups_dev, max_groups, sms, s);
}

cudaError_t launch_group_aggregate(const Plan& p, int64_t max_rows, const int64_t* ngroups_dev, int64_t max_groups,
                                   bool values_f64, int sms, cudaStream_t s) {
  if (max_rows == 0 || max_groups == 0) return cudaSuccess;
  return values_f64 ? launch_agg_f<true>(p, max_rows, ngroups_dev, max_groups, sms, s)
                    : launch_agg_f<false>(p, max_rows, ngroups_dev, max_groups, sms, s);
}

}  // namespace ocl
