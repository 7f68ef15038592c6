// exchange.cu — hash partitioning of partial group tables for the all-to-all merge
// (SURVEY §8(f) NEXT-2).
//
// The paper is single-device; multi-device execution is its stated future work
// (PAPER.md L1240-1248), and for hashing it suggests partitioning instead of one
// global table (L793-796).  With many groups an allgather of whole partial tables
// makes every rank receive (P-1) x G_r rows; routing each partial row to the rank
// that owns its key's hash partition makes every rank receive only ~G / P rows, merge
// them, and own that partition of the result.
//
// Destination of a key: ((fmix64(key) & 0xFFFFFFFF) * P) >> 32 — the LOW hash bits,
// independent of the top bits that pick a key's start slot in the merge table
// (common.cuh), so a rank's share of the keys still spreads over its whole table.
//
// k_route_count: per-destination row counts (CTA histogram in shared memory, one
// global atomic per destination per CTA).  k_route_scatter: exclusive offsets from the
// counts (each CTA, P <= 1024 entries), then every row is copied to
// out[offset[d] + atomicAdd(cursor[d])] — rows of one destination are contiguous
// (order inside a destination is unspecified; the merge does not depend on it, up to
// fp64 summation order).
#include "launch.cuh"

namespace ocl {

constexpr int kRouteThreads = 256;
constexpr int kMaxRouteParts = 1024;

__device__ __forceinline__ uint32_t route_of(uint64_t key, uint32_t nparts) {
  return (uint32_t)(((fmix64(key) & 0xFFFFFFFFULL) * nparts) >> 32);
}

__global__ void __launch_bounds__(kRouteThreads) k_route_count(const uint8_t* rows, const int64_t* nrows_dev,
                                                               int64_t max_rows, int32_t row_bytes, uint32_t nparts,
                                                               unsigned long long* counts) {
  __shared__ uint32_t hist[kMaxRouteParts];
  for (uint32_t i = threadIdx.x; i < nparts; i += blockDim.x) hist[i] = 0;
  __syncthreads();
  const int64_t n = nrows_dev ? min(*nrows_dev, max_rows) : max_rows;
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  // warp-uniform trip count; lanes with equal destinations add once (__match_any_sync)
  for (int64_t r0 = blockIdx.x * (int64_t)blockDim.x + (threadIdx.x & ~31); r0 < n; r0 += stride) {
    const int64_t r = r0 + (threadIdx.x & 31);
    const bool ok = r < n;
    const uint32_t d = ok ? route_of(*(const uint64_t*)(rows + r * row_bytes), nparts) : 0xFFFFFFFFu;
    const uint32_t peers = __match_any_sync(0xffffffffu, d);
    if (ok && (threadIdx.x & 31) == __ffs(peers) - 1) atomicAdd(&hist[d], (uint32_t)__popc(peers));
  }
  __syncthreads();
  for (uint32_t i = threadIdx.x; i < nparts; i += blockDim.x)
    if (hist[i]) atomicAdd(&counts[i], (unsigned long long)hist[i]);
}

__global__ void __launch_bounds__(kRouteThreads) k_route_scatter(const uint8_t* rows, const int64_t* nrows_dev,
                                                                 int64_t max_rows, int32_t row_bytes, uint32_t nparts,
                                                                 const unsigned long long* counts,
                                                                 unsigned long long* cursor, uint8_t* out,
                                                                 int64_t* part_counts) {
  __shared__ unsigned long long off[kMaxRouteParts];
  if (threadIdx.x == 0) {                      // exclusive offsets (P is small)
    unsigned long long o = 0;
    for (uint32_t i = 0; i < nparts; ++i) {
      off[i] = o;
      o += counts[i];
    }
  }
  __syncthreads();
  if (blockIdx.x == 0)
    for (uint32_t i = threadIdx.x; i < nparts; i += blockDim.x) part_counts[i] = (int64_t)counts[i];
  const int64_t n = nrows_dev ? min(*nrows_dev, max_rows) : max_rows;
  const int words = row_bytes / 8;
  for (int64_t r = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; r < n; r += (int64_t)gridDim.x * blockDim.x) {
    const uint64_t* src = (const uint64_t*)(rows + r * row_bytes);
    const uint32_t d = route_of(src[0], nparts);
    const unsigned long long at = off[d] + atomicAdd(&cursor[d], 1ULL);
    uint64_t* dst = (uint64_t*)(out + (int64_t)at * row_bytes);
    for (int w = 0; w < words; ++w) dst[w] = src[w];
  }
}

size_t route_ws_bytes(int32_t nparts) { return 2 * (((size_t)nparts * 8 + 255) / 256 * 256); }

int route_max_parts() { return kMaxRouteParts; }

cudaError_t launch_route(const void* rows, const int64_t* nrows_dev, int64_t max_rows, int32_t row_bytes,
                         int32_t nparts, void* out, int64_t* part_counts, void* ws, int sms, cudaStream_t s) {
  cudaError_t e = cudaMemsetAsync(ws, 0, route_ws_bytes(nparts), s);
  if (e != cudaSuccess) return e;
  unsigned long long* counts = (unsigned long long*)ws;
  unsigned long long* cursor = (unsigned long long*)((uint8_t*)ws + route_ws_bytes(nparts) / 2);
  int64_t grid = (max_rows + kRouteThreads - 1) / kRouteThreads;
  if (grid > (int64_t)sms * 4) grid = (int64_t)sms * 4;
  if (grid < 1) grid = 1;
  count_launch(2);
  k_route_count<<<(int)grid, kRouteThreads, 0, s>>>((const uint8_t*)rows, nrows_dev, max_rows, row_bytes,
                                                     (uint32_t)nparts, counts);
  k_route_scatter<<<(int)grid, kRouteThreads, 0, s>>>((const uint8_t*)rows, nrows_dev, max_rows, row_bytes,
                                                       (uint32_t)nparts, counts, cursor, (uint8_t*)out, part_counts);
  return cudaGetLastError();
}

}  // namespace ocl
