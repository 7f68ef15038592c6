// select.cu — K1 predicate -> bitmap and K2 bitmap combination.
//
// Paper: selection encodes its result as a bitmap, each thread evaluating the
// predicate on a small chunk of the input — eight 4-byte values per thread,
// one result byte (§4.1.1); complex predicates combine
// bitmaps with bit operations (L435-438).
//
// B200 design: a warp owns a tile of 1024 rows (= 32 output words).  Lane l
// issues 128-bit loads of chunks l, l+32, ... so every warp-wide load reads 512
// contiguous bytes (coalesced; the paper's GPU access pattern, L619-633 §4.2).
// A 16-byte chunk holds R = 16/width rows -> R predicate bits; K = 32/R
// neighbouring lanes OR their bits into one 32-bit word with shuffles, and one
// shuffle round moves word j to lane j so the 32 words leave as one 128-byte
// coalesced store.  HBM-bound: bytes/row = width + 1/8.
#include "launch.cuh"

namespace ocl {


template <int W>
__device__ __forceinline__ uint32_t chunk_bits(const SelParams& p, uint4 v) {
  uint32_t b = 0;
  if constexpr (W == 1) {
    // four bytes per SIMD compare: 0xFF per byte in range, then gather the four byte
    // flags into four bits with one multiply (bit 0 of byte i lands on bit 24+i)
    const uint32_t lo4 = (uint32_t)p.lo32 * 0x01010101u, hi4 = (uint32_t)p.hi32 * 0x01010101u;
    const uint32_t w4[4] = {v.x, v.y, v.z, v.w};
#pragma unroll
    for (int i = 0; i < 4; ++i) {
      uint32_t f = __vcmpgeu4(w4[i], lo4) & __vcmpleu4(w4[i], hi4) & 0x01010101u;
      b |= ((f * 0x01020408u) >> 24) << (4 * i);
    }
  } else if constexpr (W == 4) {
    int32_t x4[4] = {(int32_t)v.x, (int32_t)v.y, (int32_t)v.z, (int32_t)v.w};
#pragma unroll
    for (int i = 0; i < 4; ++i) b |= (uint32_t)(x4[i] >= p.lo32 && x4[i] <= p.hi32) << i;
  } else {
    uint64_t u0 = ((uint64_t)v.y << 32) | v.x, u1 = ((uint64_t)v.w << 32) | v.z;
    if (p.is_f64) {
      double d0 = __longlong_as_double((long long)u0), d1 = __longlong_as_double((long long)u1);
      b = (uint32_t)(d0 >= p.flo && d0 <= p.fhi) | ((uint32_t)(d1 >= p.flo && d1 <= p.fhi) << 1);
    } else {
      b = (uint32_t)((int64_t)u0 >= p.lo && (int64_t)u0 <= p.hi) |
          ((uint32_t)((int64_t)u1 >= p.lo && (int64_t)u1 <= p.hi) << 1);
    }
  }
  constexpr int R = 16 / W;
  if (p.anti) b = ~b & ((R == 32) ? 0xFFFFFFFFu : ((1u << R) - 1));
  return b;
}

__device__ __forceinline__ bool row_pred_scalar(const SelParams& p, int64_t r) {
  bool ok;
  if (p.is_f64) {
    double d = __ldg((const double*)p.col + r);
    ok = d >= p.flo && d <= p.fhi;
  } else {
    int64_t x;
    if (p.dtype == OCL_U8) x = __ldg((const uint8_t*)p.col + r);
    else if (p.dtype == OCL_I32) x = __ldg((const int32_t*)p.col + r);
    else x = __ldg((const long long*)p.col + r);
    ok = x >= p.lo && x <= p.hi;
  }
  return ok != (bool)p.anti;
}

// One 1024-row tile whose 16-byte chunks v[] are loaded: lane `lane` gets word `lane`.
template <int W>
__device__ __forceinline__ uint32_t tile_word(const SelParams& p, const uint4 (&v)[2 * W], int lane) {
  constexpr int R = 16 / W;          // rows per 16-byte chunk
  constexpr int K = 32 / R;          // lanes per output word
  constexpr int U = 2 * W;           // chunks per lane per 1024-row tile
  uint32_t mine = 0;
#pragma unroll
  for (int u = 0; u < U; ++u) {
    uint32_t w = chunk_bits<W>(p, v[u]) << ((lane % K) * R);
#pragma unroll
    for (int o = 1; o < K; o <<= 1) w |= __shfl_xor_sync(0xffffffffu, w, o);
    uint32_t val = __shfl_sync(0xffffffffu, w, (lane % R) * K);
    if (lane / R == u) mine = val;
  }
  return mine;
}

// M consecutive 1024-row tiles per warp iteration, all their loads in flight first (M = 4
// for 1-byte columns: 2 chunks per lane per tile alone left too few bytes in flight).
template <int W, int M>
__global__ void __launch_bounds__(256) k_select_bitmap(const __grid_constant__ SelParams p) {
  constexpr int U = 2 * W;
  const int lane = threadIdx.x & 31;
  const int64_t warp = (blockIdx.x * (int64_t)blockDim.x + threadIdx.x) >> 5;
  const int64_t nwarps = ((int64_t)gridDim.x * blockDim.x) >> 5;
  const int64_t tiles = (p.n + 1023) >> 10;
  const int64_t words = (p.n + 31) >> 5;
  for (int64_t t0 = warp * M; t0 < tiles; t0 += nwarps * M) {
    if (p.vec_ok && ((t0 + M) << 10) <= p.n) {
      uint4 v[M][U];
#pragma unroll
      for (int i = 0; i < M; ++i) {
        const uint4* src = (const uint4*)((const uint8_t*)p.col + ((t0 + i) << 10) * W);
#pragma unroll
        for (int u = 0; u < U; ++u) v[i][u] = __ldcs(src + lane + 32 * u);   // streaming: read once
      }
#pragma unroll
      for (int i = 0; i < M; ++i) p.out[((t0 + i) << 5) + lane] = tile_word<W>(p, v[i], lane);
      continue;
    }
    for (int64_t t = t0; t < t0 + M && t < tiles; ++t) {
      const int64_t row0 = t << 10;
      uint32_t mine = 0;
      if (p.vec_ok && row0 + 1024 <= p.n) {
        const uint4* src = (const uint4*)((const uint8_t*)p.col + row0 * W);
        uint4 v[U];
#pragma unroll
        for (int u = 0; u < U; ++u) v[u] = __ldcs(src + lane + 32 * u);
        mine = tile_word<W>(p, v, lane);
      } else {
        // ragged tail or unaligned column: lane j evaluates the 32 rows of word j
        for (int bit = 0; bit < 32; ++bit) {
          int64_t r = row0 + 32 * lane + bit;
          if (r < p.n && row_pred_scalar(p, r)) mine |= 1u << bit;
        }
      }
      int64_t wi = (t << 5) + lane;
      if (wi < words) p.out[wi] = mine;
    }
  }
}

__device__ __forceinline__ uint32_t combine_op(int op, uint32_t x, uint32_t y) {
  return op == 0 ? (x & y) : (op == 1 ? (x | y) : (x & ~y));
}

// 16-byte vectors (4 words) per thread and iteration, 4 vectors in flight; the
// last word is masked to n (bits past n are zero, s1).
__global__ void __launch_bounds__(256) k_bitmap_combine(int op, const uint32_t* __restrict__ a,
                                                        const uint32_t* __restrict__ b, uint32_t* __restrict__ out,
                                                        int64_t n, int32_t vec) {
  const int64_t words = (n + 31) >> 5;
  const uint32_t tail_mask = (n & 31) ? ((1u << (n & 31)) - 1) : 0xFFFFFFFFu;
  int64_t done = 0;
  if (vec) {
    constexpr int U = 4;
    const int64_t nv = words >> 2;
    const uint4* a4 = (const uint4*)a;
    const uint4* b4 = (const uint4*)b;
    uint4* o4 = (uint4*)out;
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    for (int64_t v0 = blockIdx.x * (int64_t)blockDim.x * U + threadIdx.x; v0 < nv; v0 += stride * U) {
      uint4 x[U], y[U];
#pragma unroll
      for (int u = 0; u < U; ++u) {
        const int64_t v = v0 + (int64_t)u * blockDim.x;
        if (v < nv) {
          x[u] = __ldcs(a4 + v);
          y[u] = __ldcs(b4 + v);
        }
      }
#pragma unroll
      for (int u = 0; u < U; ++u) {
        const int64_t v = v0 + (int64_t)u * blockDim.x;
        if (v < nv) {
          uint4 r = make_uint4(combine_op(op, x[u].x, y[u].x), combine_op(op, x[u].y, y[u].y),
                               combine_op(op, x[u].z, y[u].z), combine_op(op, x[u].w, y[u].w));
          if (4 * v + 3 == words - 1) r.w &= tail_mask;
          __stcs(o4 + v, r);
        }
      }
    }
    done = nv * 4;
  }
  for (int64_t w = done + blockIdx.x * (int64_t)blockDim.x + threadIdx.x; w < words;
       w += (int64_t)gridDim.x * blockDim.x) {
    uint32_t x = __ldg(a + w), y = __ldg(b + w);
    uint32_t v = op == 0 ? (x & y) : (op == 1 ? (x | y) : (x & ~y));
    if (w == words - 1) v &= tail_mask;
    out[w] = v;
  }
}

// ---------------------------------------------------------------- host launchers
cudaError_t launch_select_bitmap(const SelParams& p0, int grid, cudaStream_t s) {
  if (p0.n == 0) return cudaSuccess;
  SelParams p = p0;
  if (p.dtype == OCL_U8 || p.dtype == OCL_I32) {   // clamp the int64 bounds to the column's value range
    const int64_t tmin = p.dtype == OCL_U8 ? 0 : INT32_MIN, tmax = p.dtype == OCL_U8 ? 255 : INT32_MAX;
    if (p.lo > tmax || p.hi < tmin || p.lo > p.hi) {
      p.lo32 = 1;
      p.hi32 = 0;
    } else {
      p.lo32 = (int32_t)(p.lo < tmin ? tmin : p.lo);
      p.hi32 = (int32_t)(p.hi > tmax ? tmax : p.hi);
    }
  }
  int64_t tiles = (p.n + 1023) >> 10;
  const int W = dtype_width(p.dtype);
  const int M = W == 1 ? 4 : 1;            // tiles per warp iteration
  int64_t g = ((tiles + M - 1) / M + 7) / 8;   // 8 warps per block
  if (g > grid) g = grid;
  switch (W) {
    case 1: { count_launch(); k_select_bitmap<1, 4><<<(int)g, 256, 0, s>>>(p); break; }
    case 4: { count_launch(); k_select_bitmap<4, 1><<<(int)g, 256, 0, s>>>(p); break; }
    default: { count_launch(); k_select_bitmap<8, 1><<<(int)g, 256, 0, s>>>(p); break; }
  }
  return cudaGetLastError();
}

cudaError_t launch_bitmap_combine(int op, const uint32_t* a, const uint32_t* b, uint32_t* out, int64_t n, int grid,
                                  cudaStream_t s) {
  if (n == 0) return cudaSuccess;
  int64_t words = (n + 31) >> 5;
  const int vec = ((uintptr_t)a % 16 == 0) && ((uintptr_t)b % 16 == 0) && ((uintptr_t)out % 16 == 0);
  int64_t g = (words + 1023) / 1024;
  if (g > grid) g = grid;
  count_launch();
  k_bitmap_combine<<<(int)g, 256, 0, s>>>(op, a, b, out, n, vec);
  return cudaGetLastError();
}

}  // namespace ocl
