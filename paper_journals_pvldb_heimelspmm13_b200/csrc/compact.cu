// compact.cu — K3 bitmap -> ascending TID (oid) list, single pass.
//
// Paper (§4.1.2): "First, we compute a prefix sum [33] over
// bit counts to get unique write offsets for each thread.  Then, each thread
// writes the positions of set bits within its assigned bitmap chunk to its
// corresponding offset."
//
// B200 design: one pass with a decoupled look-back scan.  A CTA (8 warps)
// claims tiles of 2048 words (65,536 rows) in order from an atomic counter, so
// every predecessor tile is owned by a running CTA (forward progress).  Per
// tile: popcounts -> warp/CTA scan -> publish the tile aggregate -> warp 0 looks
// back over predecessors' {flag|value} words (32 at a time) -> publish the
// inclusive prefix.  Oids are written word by word: the set bits of one word
// go out as one contiguous (coalesced) run of the warp's lanes.
#include "launch.cuh"

namespace ocl {

constexpr int kCompactWarps = 8;
constexpr int kCompactRounds = 8;                                     // words per lane per tile
constexpr int kCompactTileWords = kCompactWarps * 32 * kCompactRounds; // 2048
constexpr uint64_t kFlagAgg = 1ULL << 62, kFlagIncl = 2ULL << 62, kValMask = (1ULL << 62) - 1;

__device__ __forceinline__ uint64_t ld_acquire(const uint64_t* p) {
  uint64_t v;
  asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}
__device__ __forceinline__ void st_release(uint64_t* p, uint64_t v) {
  asm volatile("st.release.gpu.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}

__global__ void __launch_bounds__(kCompactWarps * 32)
    k_prefix_compact(const uint32_t* __restrict__ bitmap, int64_t n, uint32_t* __restrict__ oids,
                     int64_t* m_out, unsigned long long* tile_counter, uint64_t* status, int64_t ntiles) {
  __shared__ uint32_t warp_tot[kCompactWarps];
  __shared__ uint64_t sh_tile, sh_excl;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const int64_t words = (n + 31) >> 5;
  for (;;) {
    if (threadIdx.x == 0) sh_tile = atomicAdd(tile_counter, 1ULL);
    __syncthreads();
    const int64_t tile = (int64_t)sh_tile;
    if (tile >= ntiles) break;
    const int64_t w0 = tile * kCompactTileWords + (int64_t)warp * 32 * kCompactRounds;
    uint32_t wd[kCompactRounds];
    uint32_t lane_tot = 0;
#pragma unroll
    for (int r = 0; r < kCompactRounds; ++r) {
      int64_t wi = w0 + 32 * r + lane;
      wd[r] = wi < words ? __ldcs(bitmap + wi) : 0u;
      if (wi == words - 1 && (n & 31)) wd[r] &= (1u << (n & 31)) - 1;   // ignore tail bits
      lane_tot += __popc(wd[r]);
    }
    uint32_t wt = __reduce_add_sync(0xffffffffu, lane_tot);
    if (lane == 0) warp_tot[warp] = wt;
    __syncthreads();
    uint32_t warp_base = 0, tile_agg = 0;
#pragma unroll
    for (int w = 0; w < kCompactWarps; ++w) {
      uint32_t t = warp_tot[w];
      warp_base += (w < warp) ? t : 0;
      tile_agg += t;
    }
    if (warp == 0) {
      // publish aggregate, then look back
      uint64_t excl = 0;
      if (tile == 0) {
        if (lane == 0) st_release(status, kFlagIncl | tile_agg);
      } else {
        if (lane == 0) st_release(status + tile, kFlagAgg | tile_agg);
        int64_t pos = tile - 1;
        for (;;) {
          int64_t idx = pos - lane;
          uint64_t s = 0;
          if (idx >= 0) {
            do { s = ld_acquire(status + idx); } while ((s >> 62) == 0);
          } else {
            s = kFlagIncl;   // before tile 0: inclusive prefix 0
          }
          uint32_t incl_mask = __ballot_sync(0xffffffffu, (s >> 62) == 2);
          int first = incl_mask ? __ffs(incl_mask) - 1 : 32;
          uint64_t contrib = (lane <= first) ? (s & kValMask) : 0;
          // 64-bit warp sum
          for (int o = 16; o > 0; o >>= 1) contrib += __shfl_xor_sync(0xffffffffu, contrib, o);
          excl += contrib;
          if (first < 32) break;
          pos -= 32;
        }
        if (lane == 0) st_release(status + tile, kFlagIncl | (excl + tile_agg));
      }
      if (lane == 0) {
        sh_excl = excl;
        if (tile == ntiles - 1) *m_out = (int64_t)(excl + tile_agg);
      }
    }
    __syncthreads();
    // scatter, word by word: for word i the warp's ballot of "bit lane set" is the
    // word itself, so lane l's rank among the set bits is popc(word & lanemask_lt)
    // and the warp's set rows leave as one contiguous (coalesced) store run.
    uint64_t out_base = sh_excl + warp_base;
    const uint32_t lt = (1u << lane) - 1;
#pragma unroll
    for (int r = 0; r < kCompactRounds; ++r) {
      const uint32_t row0 = (uint32_t)((w0 + 32 * r) << 5) + lane;
#pragma unroll 8
      for (int i = 0; i < 32; ++i) {
        const uint32_t w = __shfl_sync(0xffffffffu, wd[r], i);
        if ((w >> lane) & 1u) __stcs(oids + out_base + __popc(w & lt), row0 + 32u * i);
        out_base += __popc(w);
      }
    }
    __syncthreads();
  }
}

size_t prefix_compact_ws_bytes(int64_t n) {
  int64_t words = (n + 31) >> 5;
  int64_t ntiles = (words + kCompactTileWords - 1) / kCompactTileWords;
  return 256 + (size_t)ntiles * 8;
}

cudaError_t launch_prefix_compact(const uint32_t* bitmap, int64_t n, uint32_t* oids, int64_t* m_out, void* ws,
                                  int grid, cudaStream_t s) {
  if (n == 0) return cudaMemsetAsync(m_out, 0, sizeof(int64_t), s);
  int64_t words = (n + 31) >> 5;
  int64_t ntiles = (words + kCompactTileWords - 1) / kCompactTileWords;
  cudaError_t e = cudaMemsetAsync(ws, 0, prefix_compact_ws_bytes(n), s);
  if (e != cudaSuccess) return e;
  unsigned long long* counter = (unsigned long long*)ws;
  uint64_t* status = (uint64_t*)((uint8_t*)ws + 256);
  int64_t g = ntiles < grid ? ntiles : grid;
  count_launch();
  k_prefix_compact<<<(int)g, kCompactWarps * 32, 0, s>>>(bitmap, n, oids, m_out, counter, status, ntiles);
  return cudaGetLastError();
}

}  // namespace ocl
