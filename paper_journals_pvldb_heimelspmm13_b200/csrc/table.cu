// table.cu — hash-table lifecycle: dense group ids from occupied slots,
// finalisation of accumulator states into output columns (K10), group build
// (K6 + K7), projection (K4), partial-table export and multi-GPU merge (K11).
//
// Paper: the hash table yields dense group ids (§4.1.6); after
// the per-work-group aggregation "a single thread is scheduled per group to
// compute the final aggregate" (L567-568 §4.1.7).  Here one thread per table
// slot decodes the states (AVG = SUM / COUNT) and writes the dense output row.
#include <type_traits>
#include <stdlib.h>
#include "launch.cuh"
#include "rowops.cuh"

namespace ocl {

constexpr int kOccThreads = 256;
constexpr int kSortSlots = 4096;   // order_by_key in one CTA up to this many table slots

__device__ __forceinline__ bool slot_occupied(const uint8_t* table, uint64_t cap, int32_t stride, uint64_t i) {
  return *(const uint64_t*)(table + i * (uint64_t)stride) != 0;   // side entry: occupancy flag
}
__device__ __forceinline__ uint64_t slot_key(const uint8_t* table, uint64_t cap, int32_t stride, uint64_t i) {
  return i == cap ? ~0ULL : ~*(const uint64_t*)(table + i * (uint64_t)stride);
}

// ------------------------------------------------------------------ emitters
__device__ __forceinline__ void emit_slot(const EmitArgs& a, uint8_t* e, uint64_t key, int64_t g, int32_t stride) {
  if (a.kind == EMIT_FINAL) {
    emit_final(a.fin, e, key, g);
  } else if (g < a.out_capacity) {
    uint64_t* dst = (uint64_t*)(a.partial_out + g * (int64_t)stride);
    const uint64_t* src = (const uint64_t*)e;
    dst[0] = key;
    for (int w = 1; w < stride / 8; ++w) dst[w] = src[w];
  }
}

// ------------------------------------------------------------------ occupied-slot compaction
// Pass 1: occupied slots per CTA chunk.  Pass 2: exclusive scan (one CTA).
// Pass 3: ordered rank inside each chunk -> emit.  Deterministic slot order.
__global__ void __launch_bounds__(kOccThreads) k_occ_count(const uint8_t* table, uint64_t cap, int32_t stride,
                                                           uint64_t chunk, uint32_t* counts) {
  const uint64_t nslots = cap + 1;
  uint64_t b0 = blockIdx.x * chunk, b1 = b0 + chunk < nslots ? b0 + chunk : nslots;
  uint32_t c = 0;
  for (uint64_t i = b0 + threadIdx.x; i < b1; i += blockDim.x) c += slot_occupied(table, cap, stride, i) ? 1u : 0u;
  c = __reduce_add_sync(0xffffffffu, c);
  __shared__ uint32_t ws[kOccThreads / 32];
  if ((threadIdx.x & 31) == 0) ws[threadIdx.x >> 5] = c;
  __syncthreads();
  if (threadIdx.x == 0) {
    uint32_t t = 0;
    for (int w = 0; w < kOccThreads / 32; ++w) t += ws[w];
    counts[blockIdx.x] = t;
  }
}

__global__ void __launch_bounds__(1024) k_occ_scan(const uint32_t* counts, int nblocks, uint64_t* offsets,
                                                   int64_t* ngroups_out, int64_t out_capacity, int32_t* status) {
  __shared__ uint64_t carry;
  __shared__ uint64_t wsum[32];
  if (threadIdx.x == 0) carry = 0;
  __syncthreads();
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  for (int base = 0; base < nblocks; base += 1024) {
    int i = base + threadIdx.x;
    uint64_t v = i < nblocks ? counts[i] : 0;
    uint64_t incl = v;
    for (int o = 1; o < 32; o <<= 1) {
      uint64_t y = __shfl_up_sync(0xffffffffu, incl, o);
      if (lane >= o) incl += y;
    }
    if (lane == 31) wsum[warp] = incl;
    __syncthreads();
    uint64_t woff = 0;
    for (int w = 0; w < warp; ++w) woff += wsum[w];
    uint64_t c0 = carry;
    if (i < nblocks) offsets[i] = c0 + woff + incl - v;
    __syncthreads();
    if (threadIdx.x == 1023) carry = c0 + woff + incl;
    __syncthreads();
  }
  if (threadIdx.x == 0) {
    if (ngroups_out) *ngroups_out = (int64_t)carry;
    if ((int64_t)carry > out_capacity) set_status(status, OCL_ERR_CAPACITY);
  }
}

__global__ void __launch_bounds__(kOccThreads) k_occ_emit(uint8_t* table, uint64_t cap, int32_t stride, uint64_t chunk,
                                                          const uint64_t* offsets, const __grid_constant__ EmitArgs a) {
  __shared__ uint32_t ws[kOccThreads / 32];
  const uint64_t nslots = cap + 1;
  uint64_t b0 = blockIdx.x * chunk, b1 = b0 + chunk < nslots ? b0 + chunk : nslots;
  uint64_t base = offsets[blockIdx.x];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  for (uint64_t s0 = b0; s0 < b1; s0 += blockDim.x) {
    uint64_t i = s0 + threadIdx.x;
    bool occ = i < b1 && slot_occupied(table, cap, stride, i);
    uint32_t bal = __ballot_sync(0xffffffffu, occ);
    if (lane == 0) ws[warp] = __popc(bal);
    __syncthreads();
    uint32_t woff = 0, tot = 0;
    for (int w = 0; w < kOccThreads / 32; ++w) {
      woff += w < warp ? ws[w] : 0;
      tot += ws[w];
    }
    if (occ) {
      int64_t g = (int64_t)(base + woff + __popc(bal & ((1u << lane) - 1)));
      emit_slot(a, table + i * (uint64_t)stride, slot_key(table, cap, stride, i), g, stride);
    }
    base += tot;
    __syncthreads();
  }
}

// order_by_key: one CTA gathers the occupied slots, bitonic-sorts (key, slot), emits.
__global__ void __launch_bounds__(1024) k_sorted_emit(uint8_t* table, uint64_t cap, int32_t stride,
                                                      int64_t* ngroups_out, int64_t out_capacity, int32_t* status,
                                                      const __grid_constant__ EmitArgs a) {
  __shared__ uint64_t skey[kSortSlots];
  __shared__ uint16_t sslot[kSortSlots];
  __shared__ uint32_t cnt;
  if (threadIdx.x == 0) cnt = 0;
  __syncthreads();
  for (uint64_t i = threadIdx.x; i <= cap; i += blockDim.x) {
    if (slot_occupied(table, cap, stride, i)) {
      uint32_t k = atomicAdd(&cnt, 1u);
      skey[k] = slot_key(table, cap, stride, i);
      sslot[k] = (uint16_t)i;
    }
  }
  __syncthreads();
  const uint32_t G = cnt;
  uint32_t P = 1;
  while (P < G) P <<= 1;
  for (uint32_t i = G + threadIdx.x; i < P; i += blockDim.x) {
    skey[i] = ~0ULL;
    sslot[i] = 0xFFFF;        // padding sorts after a real ~0 key (slots < kSortSlots)
  }
  __syncthreads();
  for (uint32_t k = 2; k <= P; k <<= 1) {
    for (uint32_t j = k >> 1; j > 0; j >>= 1) {
      for (uint32_t i = threadIdx.x; i < P; i += blockDim.x) {
        uint32_t ixj = i ^ j;
        if (ixj > i) {
          bool up = (i & k) == 0;
          uint64_t ka = skey[i], kb = skey[ixj];
          uint16_t sa = sslot[i], sb = sslot[ixj];
          bool gt = ka > kb || (ka == kb && sa > sb);
          if (gt == up) {
            skey[i] = kb; skey[ixj] = ka;
            sslot[i] = sb; sslot[ixj] = sa;
          }
        }
      }
      __syncthreads();
    }
  }
  for (uint32_t g = threadIdx.x; g < G; g += blockDim.x)
    emit_slot(a, table + (uint64_t)sslot[g] * stride, skey[g], g, stride);
  if (threadIdx.x == 0) {
    if (ngroups_out) *ngroups_out = G;
    if ((int64_t)G > out_capacity) set_status(status, OCL_ERR_CAPACITY);
  }
}

// Unfused aggregate finalisation: table indexed directly by gid, g < *ngroups.
__global__ void k_finalize_dense(const uint8_t* table, int32_t stride, const int64_t* ngroups, int64_t max_groups,
                                 const __grid_constant__ FinPlan f) {
  int64_t G = ngroups ? *ngroups : max_groups;
  if (G > max_groups) G = max_groups;
  for (int64_t g = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; g < G; g += (int64_t)gridDim.x * blockDim.x)
    emit_final(f, table + g * stride, 0, g);
}

// ------------------------------------------------------------------ group build (K6/K7)
// Group build in one pass (K6+K7): the CTA that claims a key's table slot
// (atomicCAS on the empty key field) also assigns its dense group id from a global
// counter (one atomicAdd per warp for all keys the warp claims) and publishes it in
// the entry's payload word as gid+1; a row that finds the key already claimed reads
// the id from there (spinning the few cycles until the claimer has written it).  A
// CTA-level direct-mapped cache in shared memory (key -> gid, 256 lines, filled
// first-come) answers repeated keys without touching HBM — for few groups every row
// after warm-up; misses probe the HBM table once per distinct key per warp
// (__match_any_sync).  Ids are dense in [0, G), order unspecified (s4).
constexpr int kGroupCache = 256;

template <int W>
__device__ __forceinline__ uint64_t ld_key(const void* p, int64_t r) {   // raw bits, zero-extended
  if constexpr (W == 1) return (uint64_t)__ldg((const uint8_t*)p + r);
  else if constexpr (W == 4) return (uint64_t)(uint32_t)__ldg((const int32_t*)p + r);
  else return (uint64_t)__ldg((const unsigned long long*)p + r);
}

// Packed key (s5) of row r; W0/W1 = key column widths known at compile time, or 0
// for the runtime-described plan.
template <int W0, int W1>
__device__ __forceinline__ uint64_t group_key(const Plan& p, int64_t r) {
  if constexpr (W0 == 0) return row_key_scalar(p, r);
  else if constexpr (W1 == 0) return ld_key<W0>(p.keys[0].col.ptr, r);
  else return ld_key<W0>(p.keys[0].col.ptr, r) << (8 * W1) | ld_key<W1>(p.keys[1].col.ptr, r);
}

// Slot of key in the table, claiming an empty one; *won = this call claimed it.
__device__ __forceinline__ uint64_t* table_claim(uint8_t* table, uint64_t mask, uint64_t key, int32_t* status,
                                                 bool* won) {
  *won = false;
  if (key == ~0ULL) {   // side entry: the key field is an occupancy flag
    uint64_t* e = (uint64_t*)(table + (mask + 1) * 16);
    if (ld_relaxed_u64(e) == 0) *won = atomicCAS((unsigned long long*)e, 0ULL, 1ULL) == 0ULL;
    return e;
  }
  const uint64_t sk = ~key;
  uint64_t h = fmix64(key) & mask;
  for (uint64_t probe = 0; probe <= mask; ++probe) {
    uint64_t* kp = (uint64_t*)(table + h * 16);
    uint64_t cur = ld_relaxed_u64(kp);
    if (cur == sk) return kp;
    if (cur == 0) {
      cur = atomicCAS((unsigned long long*)kp, 0ULL, (unsigned long long)sk);
      if (cur == 0) {
        *won = true;
        return kp;
      }
      if (cur == sk) return kp;
    }
    h = (h + 1) & mask;
  }
  set_status(status, OCL_ERR_CAPACITY);
  return nullptr;
}

template <int W0, int W1, int R>
__global__ void __launch_bounds__(256) k_group_build(const __grid_constant__ Plan p, int32_t* gid_out,
                                                     int64_t max_rows, int64_t* ngroups, int64_t* keys_out,
                                                     int64_t out_capacity) {
  // R rows per thread per iteration: every oid load, then every (dependent) key gather, in flight.
  // Measured on the 2 x u8 Q1 keys at 600M rows (2.05 ms at R = 4, 48 registers): R = 2 / 8 / 16
  // 2.67 / 2.51 / 4.16 ms; 6 or 8 blocks per SM (40 / 32 registers) 2.11 / 2.21 ms
  __shared__ unsigned long long ck[kGroupCache];
  __shared__ int32_t cs[kGroupCache];
  for (int i = threadIdx.x; i < kGroupCache; i += blockDim.x) {
    ck[i] = 0;
    cs[i] = -1;
  }
  __syncthreads();
  const int lane = threadIdx.x & 31;
  const int64_t m = p.m_dev ? *p.m_dev : max_rows;
  const int64_t step = (int64_t)gridDim.x * blockDim.x * R;
  for (int64_t j0 = (int64_t)blockIdx.x * blockDim.x * R; j0 < m; j0 += step) {
    uint64_t key[R];
    int64_t r[R];
#pragma unroll
    for (int k = 0; k < R; ++k) {
      const int64_t j = j0 + k * (int64_t)blockDim.x + threadIdx.x;
      r[k] = j < m ? (p.oids ? (int64_t)__ldg(p.oids + j) : j) : -1;
    }
#pragma unroll
    for (int k = 0; k < R; ++k) key[k] = r[k] >= 0 ? group_key<W0, W1>(p, r[k]) : 0;
#pragma unroll
    for (int k = 0; k < R; ++k) {
      const int64_t j = j0 + k * (int64_t)blockDim.x + threadIdx.x;
      const bool act = r[k] >= 0;
      int32_t gid = -1;
      const int h = (int)((key[k] * 0x9E3779B97F4A7C15ULL) >> 56);   // cache line (multiplicative hash)
      if (act && key[k] != ~0ULL && *(volatile unsigned long long*)&ck[h] == ~key[k])
        gid = *(volatile int32_t*)&cs[h];
      const bool miss = act && gid < 0;
      const unsigned mmask = __ballot_sync(0xffffffffu, miss);
      if (miss) {
        const unsigned peers = __match_any_sync(mmask, key[k]);
        const int leader = __ffs(peers) - 1;
        bool won = false;
        uint64_t* e = nullptr;
        if (lane == leader) e = table_claim(p.table, p.mask, key[k], p.status, &won);
        const unsigned wm = __ballot_sync(mmask, won);
        unsigned long long base = 0;
        if (wm) {
          const int first = __ffs(wm) - 1;
          if (lane == first) base = atomicAdd((unsigned long long*)ngroups, (unsigned long long)__popc(wm));
          base = __shfl_sync(mmask, base, first);
        }
        if (lane == leader && e) {
          int64_t g;
          if (won) {
            g = (int64_t)base + __popc(wm & ((1u << lane) - 1));
            *(volatile uint64_t*)(e + 1) = (uint64_t)g + 1;
            if (g < out_capacity) {
              if (keys_out) keys_out[g] = (int64_t)key[k];
            } else {
              set_status(p.status, OCL_ERR_CAPACITY);
            }
          } else {
            uint64_t v;
            while ((v = *(volatile uint64_t*)(e + 1)) == 0) {
            }
            g = (int64_t)v - 1;
          }
          gid = (int32_t)g;
          // publish key -> gid in the CTA cache; a reader that sees the key before the gid
          // still reads -1 and takes the miss path (correct, just not cached).  The gid is
          // written with an atomic so the publication is race-free (compute-sanitizer racecheck)
          if (key[k] != ~0ULL && atomicCAS(&ck[h], 0ULL, (unsigned long long)~key[k]) == 0ULL)
            atomicExch(&cs[h], gid);
        }
        gid = __shfl_sync(peers, gid, leader);
      }
      if (act) gid_out[j] = gid;
    }
  }
}

// ------------------------------------------------------------------ projection (K4)
// U oids per thread and iteration: the oid loads, then the dependent column loads,
// are all in flight before the first store.
template <class T>
__global__ void __launch_bounds__(256) k_gather(const T* __restrict__ col, const uint32_t* __restrict__ oids,
                                                const int64_t* m_dev, int64_t max_m, T* __restrict__ out) {
  constexpr int U = 4;
  int64_t m = m_dev ? *m_dev : max_m;
  if (m > max_m) m = max_m;
  const int64_t stride = (int64_t)gridDim.x * blockDim.x * U;
  for (int64_t j0 = blockIdx.x * (int64_t)blockDim.x * U + threadIdx.x; j0 < m; j0 += stride) {
    uint32_t r[U];
    T v[U];
#pragma unroll
    for (int u = 0; u < U; ++u) {
      const int64_t j = j0 + (int64_t)u * blockDim.x;
      r[u] = j < m ? __ldcs(oids + j) : 0u;
    }
#pragma unroll
    for (int u = 0; u < U; ++u)
      if (j0 + (int64_t)u * blockDim.x < m) v[u] = __ldg(col + r[u]);
#pragma unroll
    for (int u = 0; u < U; ++u) {
      const int64_t j = j0 + (int64_t)u * blockDim.x;
      if (j < m) __stcs(out + j, v[u]);
    }
  }
}

// ------------------------------------------------------------------ merge partials (K11)
__global__ void k_merge_partials(const uint8_t* partials, int32_t nparts, int64_t part_capacity,
                                 const int64_t* part_counts, const __grid_constant__ FinPlan f, uint8_t* table,
                                 uint64_t mask, int32_t* status) {
  const int32_t stride = f.stride;
  for (int32_t part = 0; part < nparts; ++part) {
    int64_t cnt = part_counts[part];
    if (cnt > part_capacity) cnt = part_capacity;
    for (int64_t j = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; j < cnt; j += (int64_t)gridDim.x * blockDim.x) {
      const uint8_t* row = partials + ((int64_t)part * part_capacity + j) * stride;
      uint64_t key = *(const uint64_t*)row;
      uint8_t* e = table_find_or_insert(table, mask, stride, key, status);
      if (!e) continue;
      atomicAdd((unsigned long long*)(e + 8), *(const unsigned long long*)(row + 8));
      for (int s = 0; s < f.nstates; ++s) {
        const StateDesc& d = f.states[s];
        const uint8_t* src = row + d.off;
        uint8_t* dst = e + d.off;
        if (d.kind == ACC_SUM_I) atomic_add_i128((uint64_t*)dst, *(const uint64_t*)src, *(const uint64_t*)(src + 8));
        else if (d.kind == ACC_SUM_F) atomicAdd((double*)dst, *(const double*)src);
        else atomicMax((unsigned long long*)dst, *(const unsigned long long*)src);
      }
    }
  }
}

// ------------------------------------------------------------------ host launchers
static uint64_t occ_chunk(uint64_t nslots, int grid, int* nblocks) {
  uint64_t chunk = (nslots + grid - 1) / grid;
  chunk = (chunk + kOccThreads - 1) / kOccThreads * kOccThreads;
  if (chunk < kOccThreads) chunk = kOccThreads;
  *nblocks = (int)((nslots + chunk - 1) / chunk);
  return chunk;
}

size_t emit_ws_bytes(int grid) { return (size_t)grid * 16 + 256; }

// Emit all occupied slots of a table (cap = mask + 1) in slot order (or key order).
cudaError_t launch_emit(uint8_t* table, uint64_t cap, int32_t stride, const EmitArgs& a, int64_t* ngroups_out,
                        int64_t out_capacity, int32_t* status, bool sorted, void* ws, int grid, cudaStream_t s) {
  if (sorted) {
    if (cap + 1 > (uint64_t)kSortSlots) return cudaErrorInvalidValue;
    count_launch();
    k_sorted_emit<<<1, 1024, 0, s>>>(table, cap, stride, ngroups_out, out_capacity, status, a);
    return cudaGetLastError();
  }
  int nblocks = 0;
  uint64_t chunk = occ_chunk(cap + 1, grid, &nblocks);
  uint32_t* counts = (uint32_t*)ws;
  uint64_t* offsets = (uint64_t*)((uint8_t*)ws + (((size_t)grid * 4 + 255) / 256) * 256);
  count_launch();
  k_occ_count<<<nblocks, kOccThreads, 0, s>>>(table, cap, stride, chunk, counts);
  count_launch();
  k_occ_scan<<<1, 1024, 0, s>>>(counts, nblocks, offsets, ngroups_out, out_capacity, status);
  count_launch();
  k_occ_emit<<<nblocks, kOccThreads, 0, s>>>(table, cap, stride, chunk, offsets, a);
  return cudaGetLastError();
}

bool sorted_emit_supported(uint64_t cap) { return cap + 1 <= (uint64_t)kSortSlots; }

cudaError_t launch_finalize_dense(const uint8_t* table, int32_t stride, const int64_t* ngroups, int64_t max_groups,
                                  const FinPlan& f, int grid, cudaStream_t s) {
  if (max_groups == 0) return cudaSuccess;
  int64_t g = (max_groups + 255) / 256;
  if (g > grid) g = grid;
  count_launch();
  k_finalize_dense<<<(int)g, 256, 0, s>>>(table, stride, ngroups, max_groups, f);
  return cudaGetLastError();
}

cudaError_t launch_group_build(const Plan& p, int32_t* gid_out, int64_t max_rows, int64_t* ngroups,
                               int64_t* keys_out, int64_t out_capacity, int grid, cudaStream_t s) {
  if (max_rows == 0) return cudaSuccess;
  int64_t g = (max_rows + 1023) / 1024;
  if (g > grid) g = grid;
  const char* er = getenv("OCL_GB_R");
  const int rr = er ? atoi(er) : 4;
  auto pick = [&](auto r) {
    constexpr int R = decltype(r)::value;
    auto fn = k_group_build<0, 0, R>;
    const int w0 = p.keys[0].col.width, w1 = p.nkeys > 1 ? p.keys[1].col.width : 0;
    if (p.nkeys == 2 && w0 == 1 && w1 == 1) fn = k_group_build<1, 1, R>;
    else if (p.nkeys == 2 && w0 == 4 && w1 == 4) fn = k_group_build<4, 4, R>;
    else if (p.nkeys == 1 && w0 == 1) fn = k_group_build<1, 0, R>;
    else if (p.nkeys == 1 && w0 == 4) fn = k_group_build<4, 0, R>;
    else if (p.nkeys == 1 && w0 == 8) fn = k_group_build<8, 0, R>;
    return fn;
  };
  auto fn = rr >= 16 ? pick(std::integral_constant<int, 16>{})
            : rr >= 8 ? pick(std::integral_constant<int, 8>{})
            : rr <= 2 ? pick(std::integral_constant<int, 2>{}) : pick(std::integral_constant<int, 4>{});
  count_launch();
  fn<<<(int)g, 256, 0, s>>>(p, gid_out, max_rows, ngroups, keys_out, out_capacity);
  return cudaGetLastError();
}

cudaError_t launch_gather(const void* col, int32_t width, const uint32_t* oids, const int64_t* m_dev, int64_t max_m,
                          void* out, int grid, cudaStream_t s) {
  if (max_m == 0) return cudaSuccess;
  int64_t g = (max_m + 1023) / 1024;
  if (g > grid) g = grid;
  count_launch();
  if (width == 1) k_gather<uint8_t><<<(int)g, 256, 0, s>>>((const uint8_t*)col, oids, m_dev, max_m, (uint8_t*)out);
  else if (width == 4) k_gather<int32_t><<<(int)g, 256, 0, s>>>((const int32_t*)col, oids, m_dev, max_m, (int32_t*)out);
  else k_gather<long long><<<(int)g, 256, 0, s>>>((const long long*)col, oids, m_dev, max_m, (long long*)out);
  return cudaGetLastError();
}

cudaError_t launch_merge_partials(const uint8_t* partials, int32_t nparts, int64_t part_capacity,
                                  const int64_t* part_counts, const FinPlan& f, uint8_t* table, uint64_t mask,
                                  int32_t* status, int grid, cudaStream_t s) {
  if (nparts == 0 || part_capacity == 0) return cudaSuccess;
  int64_t g = (part_capacity + 255) / 256;
  if (g > grid) g = grid;
  count_launch();
  k_merge_partials<<<(int)g, 256, 0, s>>>(partials, nparts, part_capacity, part_counts, f, table, mask, status);
  return cudaGetLastError();
}

}  // namespace ocl
