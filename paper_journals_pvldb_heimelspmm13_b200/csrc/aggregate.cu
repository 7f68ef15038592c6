// aggregate.cu — K8: grouped aggregation over a dense group-id column (unfused chain).
//
// Paper (§4.1.7): work-groups on disjoint partitions build
// intermediate aggregation tables with atomics in local memory; for few groups
// each group is spread over several accumulators ("the number of accumulators
// per group being chosen inversely proportional to the number of groups") to
// cut same-address contention; tables that do not fit local memory fall back to
// the same scheme in global memory.  Then one thread per group finalises.
//
// B200 design: SMEM tier — R replicas of the G-entry state table in shared memory
// (R = largest power of two <= 32 with R*G*stride <= the smem budget, lane picks
// replica lane % R), shared-memory atomics (native 64-bit add / max, fp64 add),
// then one flush of the CTA's non-empty entries into the HBM table.  GLOBAL tier
// when G*stride exceeds shared memory: the same updates on the HBM table.
// Values are read at row oids[j] (fused gather), integer expressions in int128.
#include "launch.cuh"
#include "rowops.cuh"

namespace ocl {

__device__ __forceinline__ void agg_update_row(const Plan& p, uint8_t* e, int64_t r) {
  atomicAdd((unsigned long long*)(e + 8), 1ULL);
  for (int i = 0; i < p.nvals; ++i) {
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
      bool fast = true;
      int64_t x = value_i64_fast(v, ra, rb, rc, fast);
      I128 y = fast ? i128_from_i64(x) : value_i128(v, ra, rb, rc);
      if (v.off_sum >= 0) atomic_add_i128((uint64_t*)(e + v.off_sum), y.lo, y.hi);
      if (v.off_min >= 0) atomicMax((unsigned long long*)(e + v.off_min), (unsigned long long)enc_min_i((int64_t)y.lo));
      if (v.off_max >= 0) atomicMax((unsigned long long*)(e + v.off_max), (unsigned long long)enc_max_i((int64_t)y.lo));
    }
  }
}

template <bool SMEM>
__global__ void __launch_bounds__(256) k_group_aggregate(const __grid_constant__ Plan p, int64_t max_rows,
                                                         const int64_t* ngroups_dev, int64_t max_groups,
                                                         int32_t replicas) {
  extern __shared__ __align__(16) uint64_t sm[];
  int64_t G = ngroups_dev ? *ngroups_dev : max_groups;
  if (G > max_groups) G = max_groups;
  const int64_t m = p.m_dev ? *p.m_dev : max_rows;
  const int64_t words = SMEM ? (int64_t)replicas * G * p.stride / 8 : 0;
  if constexpr (SMEM) {
    for (int64_t i = threadIdx.x; i < words; i += blockDim.x) sm[i] = 0;
    __syncthreads();
  }
  const int rep = (threadIdx.x & 31) & (replicas - 1);
  for (int64_t j = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; j < m; j += (int64_t)gridDim.x * blockDim.x) {
    int32_t g = __ldg(p.gids + j);
    if (g < 0 || g >= G) continue;
    int64_t r = p.oids ? (int64_t)__ldg(p.oids + j) : j;
    uint8_t* e = SMEM ? (uint8_t*)sm + ((int64_t)rep * G + g) * p.stride : p.table + (int64_t)g * p.stride;
    agg_update_row(p, e, r);
  }
  if constexpr (SMEM) {
    __syncthreads();
    // flush: one thread per (group, replica) entry with a non-zero count
    for (int64_t i = threadIdx.x; i < (int64_t)replicas * G; i += blockDim.x) {
      const uint8_t* se = (const uint8_t*)sm + i * p.stride;
      uint64_t c = *(const uint64_t*)(se + 8);
      if (c == 0) continue;
      uint8_t* e = p.table + (i % G) * p.stride;
      atomicAdd((unsigned long long*)(e + 8), (unsigned long long)c);
      for (int v = 0; v < p.nvals; ++v) {
        const DevValue& d = p.vals[v];
        if (d.off_sum >= 0) {
          if (d.is_f64) atomicAdd((double*)(e + d.off_sum), *(const double*)(se + d.off_sum));
          else atomic_add_i128((uint64_t*)(e + d.off_sum), *(const uint64_t*)(se + d.off_sum),
                               *(const uint64_t*)(se + d.off_sum + 8));
        }
        if (d.off_min >= 0) atomicMax((unsigned long long*)(e + d.off_min), *(const unsigned long long*)(se + d.off_min));
        if (d.off_max >= 0) atomicMax((unsigned long long*)(e + d.off_max), *(const unsigned long long*)(se + d.off_max));
      }
    }
  }
}

constexpr size_t kAggSmemBudget = 96 * 1024;

cudaError_t launch_group_aggregate(const Plan& p, int64_t max_rows, const int64_t* ngroups_dev, int64_t max_groups,
                                   int grid, cudaStream_t s) {
  if (max_rows == 0 || max_groups == 0) return cudaSuccess;
  int64_t g = (max_rows + 255) / 256;
  if (g > grid) g = grid;
  size_t one = (size_t)max_groups * p.stride;
  if (one <= kAggSmemBudget) {
    int R = 32;
    while (R > 1 && (size_t)R * one > kAggSmemBudget) R >>= 1;
    size_t bytes = (size_t)R * one;
    cudaError_t e = cudaFuncSetAttribute(k_group_aggregate<true>, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                         (int)kAggSmemBudget);
    if (e != cudaSuccess) return e;
    count_launch();
    k_group_aggregate<true><<<(int)g, 256, bytes, s>>>(p, max_rows, ngroups_dev, max_groups, R);
  } else {
    count_launch();
    k_group_aggregate<false><<<(int)g, 256, 0, s>>>(p, max_rows, ngroups_dev, max_groups, 1);
  }
  return cudaGetLastError();
}

}  // namespace ocl
