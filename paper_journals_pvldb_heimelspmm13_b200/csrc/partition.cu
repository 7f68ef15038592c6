// partition.cu — high-cardinality tier of the fused select -> group -> aggregate:
// hash-partitioned two-pass aggregation.
//
// The paper's GPU group-by inserts every row into one device-wide hash table with
// atomics and names hashing "one of the major shortcomings" (PAPER.md L949-954
// §5.2.1); for many groups the table lives in device memory and every row pays a
// random read-modify-write there (§4.1.6, §4.1.7).  It also
// suggests partitioning the work over a global hash table.  On B200 a
// random atomic into a table larger than L2 costs ~10x a streamed row
// (tools/micro/atom_bench.cu: 10.9 G rows/s for 4 atomics per row into 1 GB), while
// 32-bit shared-memory atomics on random addresses sustain ~8 per clock per SM
// (tools/micro/smem_atom_bench.cu).  So for many groups the rows are first routed by
// hash to P = 2^pbits partitions small enough for a shared-memory table:
//
//   pass 1a  k_part_count    fused select + key + values, per row-block histogram of
//                            partition ids (shared-memory counters); per row block the
//                            level-1 counts (top b1 = 7 hash bits)
//   scan     k_scan_*        exclusive scans: partition starts, per-block level-1 ranges
//   pass 1b  k_part_scatter_l1  the same rows again: each qualifying row becomes a record
//                            {key, int32 values} in its row block's own range of its
//                            level-1 partition (block-local cursors, no global claims),
//                            staged per tile in shared memory and written as runs;
//            k_part_scatter2 level-1 records -> final partitions, per tile one global
//                            claim per partition met (direct-indexed tile map).  With
//                            <= 2^7 partitions one tiled level (k_part_scatter).
//   pass 2   k_part_agg      work items of <= kPartItem records of one partition; a
//                            CTA aggregates an item in a shared-memory hash table
//                            (32-bit atomics, field-major) and emits its groups straight
//                            from shared memory (or merges them into the HBM table)
//
// The HBM table's start slot is the top bits of the key hash (common.cuh), so a
// partition's keys occupy one contiguous slot range (its region).  The table is zeroed
// lazily: only regions that receive entries (exact-path rows, split or overflowing
// partitions) are cleared.  Rows the fast path cannot take (values outside int32, the
// key ~0) and records whose partition overflows the shared table update the HBM table
// directly (exact).
#include <string.h>

#include "launch.cuh"
#include "sga_device.cuh"

namespace ocl {

constexpr int kPartThreads = 512;
constexpr int kPartCapBits = 11;
constexpr int kPartCap = 1 << kPartCapBits;   // shared-table entries per CTA in pass 2
static_assert(kPartCap == (int)kProbeWindow, "direct merges need partition ranges = HBM probe windows");
constexpr int kPartItem = 32768;      // records per pass-2 work item (<= 2^15: 16-bit split sums of the table stay exact)
constexpr int kPartILP = 4;           // rows / records per thread in flight (part_rows: 2 units x 2 rows)
constexpr int kTileMapBits = 12;      // scatter: per-tile partition map (2 x the tile's rows)
constexpr int kPartLevelBits = 7;     // partitions reached per scatter level (tile claims aggregate ~16x)
constexpr int kTileMap = 1 << kTileMapBits;
constexpr int kScanThreads = 1024;
constexpr int kScanPer = 8;           // elements per thread per scan chunk
constexpr int kScanChunk = kScanThreads * kScanPer;

struct PartArgs {
  int32_t pbits;
  int32_t nblk;
  int64_t rows_per_blk;
  uint32_t* counts;     // [P] histogram of partition ids
  uint32_t* offs;       // [P] exclusive scan of counts: partition starts
  uint32_t* cur;        // [P] global write cursors of pass 1b (start = offs)
  uint32_t* curp;       // [P << curp_shift] the same, one per 2^curp_shift words (one-level scatter:
  int32_t curp_shift;   //   a cursor per L2 sector / line, so claims on different partitions do not queue)
  uint32_t* sums;       // scan chunk sums
  int64_t* m_dev;       // number of records
  uint8_t* recs;        // records: {key u64, int32 value x NV}, rec_bytes each, grouped by partition
  uint8_t* tmp;         // level-1 records (two-level scatter), grouped by the top b1 hash bits
  uint32_t* cur1;       // [2^b1] level-1 cursors
  uint32_t* cnt1;       // [2^b1][nblk] level-1 counts per row block (count pass), then their
                        // exclusive scan: each block's own range in every level-1 partition
  uint32_t* sums1;      // scan chunk sums of cnt1
  int32_t b1;           // level-1 bits (two-level scatter)
  // low selectivity (sparse_dev != NULL and *sparse_dev = 1, decided on the device from a
  // sample): the count pass streams the predicate columns only, evaluates the other columns
  // of qualifying rows and lists their row ids in its block's range of soids (nq[block] of
  // them); the level-1 scatter reads those lists instead of the columns
  int32_t* sparse_dev;
  uint32_t* soids;      // [n] row ids, block b's list at [b * rows_per_blk, + nq[b])
  uint32_t* nq;         // [nblk]
  uint32_t* icnt;       // [P] pass-2 work items per partition
  uint32_t* ioff;       // [P] exclusive scan of icnt
  uint32_t* isums;      // scan chunk sums of icnt
  int64_t* nitems_dev;  // number of pass-2 work items
  uint32_t* slowflag;   // [P] 1: the exact path inserted keys of this partition in pass 1
  int32_t direct_ok;    // the HBM table's partition regions have exactly kPartCap slots
  int32_t rec_bytes;
  // direct emission (direct_emit = 1): partitions aggregated entirely in shared memory write
  // their output rows (final or partial) straight from there; the others mark dirty[q] and
  // are emitted from their HBM slot range afterwards — no pass over the whole table.
  int32_t direct_emit;
  // lazy = 1: the caller did not zero the HBM table; k_part_zero_regions clears the regions
  // known to be used before pass 1b, a partition whose shared table overflows clears its own
  // region and re-aggregates its item there (requires direct_emit).
  int32_t lazy;
  int32_t mm_check;     // pass 2: MIN / MAX read-before-atomic
  int32_t npo;                     // final outputs, resolved on the host (kind, CTA-entry fields, pointer)
  struct { int32_t kind, f0, f1, pad; void* out; } po[kMaxAggs];
  uint32_t* dirty;                 // [P]
  unsigned long long* out_ctr;     // output rows so far
  int64_t* count_out;              // G (or the partial row count)
};

// One output row (final or partial) from a table-format entry e (key = the real key).
__device__ __forceinline__ void part_emit_row(const EmitArgs& ea, int32_t stride, const uint8_t* e, uint64_t key,
                                              int64_t g) {
  if (ea.kind == EMIT_FINAL) {
    emit_final(ea.fin, e, key, g);
  } else if (g < ea.out_capacity) {
    uint64_t* dst = (uint64_t*)(ea.partial_out + g * (int64_t)stride);
    dst[0] = key;
    for (int w = 1; w < stride / 8; ++w) dst[w] = ((const uint64_t*)e)[w];
  }
}

// CTA: claim output positions for the `cnt` rows this thread emits (block scan + one atomic).
__device__ __forceinline__ int64_t part_emit_claim(uint32_t cnt, unsigned long long* ctr, uint32_t* wsum,
                                                   unsigned long long* base_s) {
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  uint32_t incl = cnt;
#pragma unroll
  for (int d = 1; d < 32; d <<= 1) {
    const uint32_t y = __shfl_up_sync(0xffffffffu, incl, d);
    if (lane >= d) incl += y;
  }
  if (lane == 31) wsum[warp] = incl;
  __syncthreads();
  uint32_t off = 0, tot = 0;
  for (int w = 0; w < (int)(blockDim.x >> 5); ++w) {
    off += w < warp ? wsum[w] : 0u;
    tot += wsum[w];
  }
  if (threadIdx.x == 0) *base_s = tot ? atomicAdd(ctr, (unsigned long long)tot) : 0ULL;
  __syncthreads();
  const int64_t g = (int64_t)(*base_s + off + incl - cnt);
  __syncthreads();
  return g;
}

__device__ __forceinline__ uint32_t part_of(uint64_t key, int pbits) {
  return pbits ? (uint32_t)(fmix64(key) >> (64 - pbits)) : 0u;
}

// Lanes whose partition equals lane 0's are served by one shared-memory atomic of
// lane 0 (hot keys of skewed data); the others each take one.  Returns the base
// position for the aggregated group (valid in lanes of `same`) via *base.
__device__ __forceinline__ uint32_t lanemask_lt() {
  uint32_t m;
  asm("mov.u32 %0, %%lanemask_lt;" : "=r"(m));
  return m;
}

template <class Sh, int NV>
__device__ __forceinline__ void part_eval(const Plan& p, int64_t r, int64_t r1, Row<Sh, NV, false>& x, bool& ok) {
  eval_one<Sh, NV, false>(p, r, x);
  x.q = x.q && r < r1;
  ok = x.q && x.fast && !Sh::special(x.key);
}

// The kPartILP = 4 rows of a lane in a tile: warp w owns the 128 rows [wbase, wbase +
// 128) as two 64-row units, lane l their rows 2l, 2l+1 (the fused kernel's layout).
// Static shapes with aligned columns load both units with vector loads, no branches,
// all loads in flight before any row is evaluated; the rest evaluate row by row.
__device__ __forceinline__ int64_t part_row(int64_t wbase, int lane, int i) {
  return wbase + (i >> 1) * 64 + 2 * lane + (i & 1);
}

template <class Sh, int NV>
__device__ __forceinline__ void part_rows(const Plan& p, int64_t wbase, int64_t r1, int lane,
                                          Row<Sh, NV, false> (&x)[4], bool (&ok)[4]) {
  if constexpr (Sh::kStatic) {
    if (p.vec_ok && wbase + 128 <= r1) {
      RawUnit<Sh> u[2];
      load_unit<Sh>(p, wbase + 2 * lane, u[0]);
      load_unit<Sh>(p, wbase + 64 + 2 * lane, u[1]);
#pragma unroll
      for (int i = 0; i < 4; ++i) {
        eval_unit<Sh, NV, false>(p, u[i >> 1], i & 1, x[i]);
        ok[i] = x[i].q && x[i].fast && !Sh::special(x[i].key);
      }
      return;
    }
  }
#pragma unroll
  for (int i = 0; i < 4; ++i) part_eval<Sh, NV>(p, part_row(wbase, lane, i), r1, x[i], ok[i]);
}

// Predicates only (row r < n): the first step of the sparse mode.
template <class Sh>
__device__ __forceinline__ bool row_qualifies(const Plan& p, int64_t r) {
  bool q = true;
#pragma unroll
  for (int i = 0; i < kMaxPreds; ++i) {
    if (i >= Sh::np(p)) break;
    q = q && pred_ok<Sh>(p, i, ld1w(Sh::pw(p, i), p.preds[i].col.ptr, r));
  }
  return q;
}

// Sparse-mode decision: the predicates on 1024 rows spread over the input (one CTA).
constexpr int kPartSparsePct = 8;     // below this many percent qualifying: sparse mode
template <class Sh>
__global__ void __launch_bounds__(1024) k_part_sample(const __grid_constant__ Plan p, int32_t* sparse_dev) {
  __shared__ int cnt;
  if (threadIdx.x == 0) cnt = 0;
  __syncthreads();
  const int64_t span = p.n / 1024;
  if (span > 0 && row_qualifies<Sh>(p, (int64_t)threadIdx.x * span)) atomicAdd(&cnt, 1);
  __syncthreads();
  if (threadIdx.x == 0) *sparse_dev = (span > 0 && 100 * cnt < kPartSparsePct * 1024) ? 1 : 0;
}

// ------------------------------------------------------------------ pass 1a: histogram
template <class Sh, int NV, bool SPARSE>
__global__ void __launch_bounds__(kPartThreads) k_part_count(const __grid_constant__ Plan p, PartArgs a) {
  // SPARSE: the low-selectivity variant, launched next to the dense one; each returns at
  // once unless the device-side sample chose its mode (grid-uniform)
  if (a.sparse_dev && (*a.sparse_dev != 0) != SPARSE) return;
  extern __shared__ uint32_t hist[];
  const int P = 1 << a.pbits;
  const int lane = threadIdx.x & 31;
  for (int i = threadIdx.x; i < P; i += blockDim.x) hist[i] = 0;
  __syncthreads();
  const int64_t r0 = blockIdx.x * a.rows_per_blk;
  const int64_t r1 = min(p.n, r0 + a.rows_per_blk);
  const int64_t woff = (int64_t)(threadIdx.x >> 5) * 128;
  constexpr bool sparse = SPARSE;
  if constexpr (SPARSE) {
    // 256 rows per warp step, lane l row base + l + 32 i: coalesced predicate loads, then
    // qualifying rows listed (warp-aggregated claim in the block's list) and evaluated
    __shared__ uint32_t blk_n;
    if (threadIdx.x == 0) blk_n = 0;
    __syncthreads();
    const uint32_t lt = lanemask_lt();
    const int64_t nwarp = blockDim.x >> 5;
    for (int64_t base = r0 + (int64_t)(threadIdx.x >> 5) * 256; base < r1; base += nwarp * 256) {
      bool q[8];
      unsigned bal[8];
      uint32_t tot = 0;
#pragma unroll
      for (int i = 0; i < 8; ++i) {
        const int64_t r = base + 32 * i + lane;
        q[i] = r < r1 && row_qualifies<Sh>(p, r);
      }
#pragma unroll
      for (int i = 0; i < 8; ++i) {
        bal[i] = __ballot_sync(0xffffffffu, q[i]);
        tot += __popc(bal[i]);
      }
      if (tot == 0) continue;
      uint32_t wb = 0;
      if (lane == 0) wb = atomicAdd(&blk_n, tot);
      wb = __shfl_sync(0xffffffffu, wb, 0);
#pragma unroll
      for (int i = 0; i < 8; ++i) {
        const int64_t r = base + 32 * i + lane;
        if (q[i]) {
          a.soids[r0 + wb + __popc(bal[i] & lt)] = (uint32_t)r;
          Row<Sh, NV, false> x;
          eval_one<Sh, NV, false>(p, r, x);
          const bool ok = x.q && x.fast && !Sh::special(x.key);
          if (ok) atomicAdd(&hist[part_of((uint64_t)x.key, a.pbits)], 1u);
          else if (x.q && (uint64_t)x.key != ~0ULL) a.slowflag[part_of((uint64_t)x.key, a.pbits)] = 1u;
        }
        wb += __popc(bal[i]);
      }
    }
    __syncthreads();
    if (threadIdx.x == 0) a.nq[blockIdx.x] = blk_n;
  }
  for (int64_t base = r0; base < (sparse ? r0 : r1); base += kPartILP * blockDim.x) {
    Row<Sh, NV, false> x[kPartILP];
    bool ok[kPartILP];
    part_rows<Sh, NV>(p, base + woff, r1, lane, x, ok);
#pragma unroll
    for (int k = 0; k < kPartILP; ++k) {
      const uint32_t part = ok[k] ? part_of((uint64_t)x[k].key, a.pbits) : 0xFFFFFFFFu;
      const uint32_t p0 = __shfl_sync(0xffffffffu, part, 0);
      const unsigned same = __ballot_sync(0xffffffffu, ok[k] && part == p0);
      if (x[k].q && !ok[k] && (uint64_t)x[k].key != ~0ULL)   // exact-path row: its region is used
        a.slowflag[part_of((uint64_t)x[k].key, a.pbits)] = 1u;
      if (ok[k] && part != p0) atomicAdd(&hist[part], 1u);
      if (lane == 0 && same) atomicAdd(&hist[p0], (uint32_t)__popc(same));
    }
  }
  __syncthreads();
  for (int i = threadIdx.x; i < P; i += blockDim.x)
    if (hist[i]) atomicAdd(&a.counts[i], hist[i]);
  if (a.cnt1) {                            // two-level scatter: this block's level-1 counts
    const int P1 = 1 << a.b1, w = 1 << (a.pbits - a.b1);
    for (int t = threadIdx.x; t < P1; t += blockDim.x) {
      uint32_t c = 0;
      for (int i = 0; i < w; ++i) c += hist[t * w + i];
      a.cnt1[(size_t)t * a.nblk + blockIdx.x] = c;
    }
  }
}

// ------------------------------------------------------------------ pass 1b: scatter
// Scatter claims, aggregated per tile of kPartILP x T rows or records: a shared-memory
// map partition -> count gives every item its rank, then one global atomic per
// distinct partition of the tile claims the range from that partition's cursor
// (shared by all CTAs).  Shared cursors keep only a couple of lines per partition
// open in L2, so the 16-byte record stores combine into full lines (per-CTA ranges
// kept P x #CTAs partial lines open, overflowed L2 and turned every store into a
// partial-sector read-modify-write: measured 2x writes, 2.4x reads).  Aggregation
// needs several items per partition per tile, so more than 128 partitions are
// reached in two levels (k_part_scatter2).
struct TileMap {
  uint32_t key[kTileMap];
  uint32_t cnt[kTileMap];                  // count, then the global base of the slot's range
  uint32_t off[kTileMap];                  // the slot's first index in the staging area
  uint16_t sslot[kPartILP * kPartThreads]; // slot of each staged item
  uint4 stage[kPartILP * kPartThreads];    // the tile's records, grouped by partition
  uint16_t used[kPartILP * kPartThreads];  // slots taken in this tile (a tile meets ~128 of the 4096)
  uint32_t nused;
  uint32_t total;                          // items in the tile
};

// Whole map empty (once per CTA; the caller synchronises).
__device__ __forceinline__ void tile_map_init(TileMap& m) {
  for (int i = threadIdx.x; i < kTileMap; i += blockDim.x) {
    m.key[i] = 0xFFFFFFFFu;
    m.cnt[i] = 0;
  }
  if (threadIdx.x == 0) m.nused = 0;
}

// Empty again after a tile: only the slots the tile used (instead of all 4096 — the
// per-tile clear and the claim scan over the whole map dominated the scatter passes).
__device__ __forceinline__ void tile_map_reset(TileMap& m) {
  const uint32_t nu = m.nused;
  __syncthreads();
  for (uint32_t i = threadIdx.x; i < nu; i += blockDim.x) {
    const uint32_t sl = m.used[i];
    m.key[sl] = 0xFFFFFFFFu;
    m.cnt[sl] = 0;
  }
  if (threadIdx.x == 0) m.nused = 0;
}

// slot of `part` in the map (inserted if new) and this item's rank within it
__device__ __forceinline__ void tile_map_add(TileMap& m, uint32_t part, uint32_t& slot, uint32_t& rank) {
  volatile uint32_t* vk = m.key;
  uint32_t h = (part * 0x9E3779B1u) >> (32 - kTileMapBits);
  while (true) {                           // < kTileMap / 2 distinct partitions per tile: terminates
    const uint32_t cur = vk[h];
    if (cur == part) break;
    if (cur == 0xFFFFFFFFu) {
      const uint32_t prev = atomicCAS(&m.key[h], 0xFFFFFFFFu, part);
      if (prev == 0xFFFFFFFFu) {
        m.used[atomicAdd(&m.nused, 1u)] = (uint16_t)h;
        break;
      }
      if (prev == part) break;
    }
    h = (h + 1) & (kTileMap - 1);
  }
  slot = h;
  rank = atomicAdd(&m.cnt[h], 1u);
}

// After a barrier: counts -> global bases, and each used slot's offset in the staging
// area (exclusive scan of the used slots' counts, 256 at a time).
__device__ __forceinline__ void tile_map_claim(TileMap& m, uint32_t* cur, uint32_t* wsum) {
  const int t = threadIdx.x, lane = t & 31, w = t >> 5;
  const uint32_t nu = m.nused;
  uint32_t run0 = 0;
  for (uint32_t b0 = 0; b0 < nu; b0 += kPartThreads) {
    const uint32_t i = b0 + t;
    const uint32_t sl = i < nu ? m.used[i] : 0u;
    const uint32_t c = i < nu ? m.cnt[sl] : 0u;
    uint32_t incl = c;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      const uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
      if (lane >= o) incl += y;
    }
    if (lane == 31) wsum[w] = incl;
    __syncthreads();
    uint32_t off = 0, tot = 0;
#pragma unroll
    for (int k = 0; k < kPartThreads / 32; ++k) {
      off += k < w ? wsum[k] : 0u;
      tot += wsum[k];
    }
    if (i < nu) {
      m.off[sl] = run0 + off + incl - c;
      m.cnt[sl] = atomicAdd(&cur[m.key[sl]], c);
    }
    run0 += tot;
    __syncthreads();
  }
  if (t == 0) m.total = run0;
}

// Direct-indexed variant (slot i = partition qb + i, i < width): the same claim over every
// slot of the range instead of the used list; bases go to gb[] and the counters are left
// zeroed (no reset pass after the flush).
constexpr uint32_t kDirectMap = 1024;
__device__ __forceinline__ void tile_dmap_claim(TileMap& m, uint32_t width, uint32_t qb, uint32_t* cur,
                                                uint32_t* wsum, uint32_t* gb) {
  const int t = threadIdx.x, lane = t & 31, w = t >> 5;
  uint32_t run0 = 0;
  for (uint32_t b0 = 0; b0 < width; b0 += kPartThreads) {
    const uint32_t i = b0 + t;
    const uint32_t c = i < width ? m.cnt[i] : 0u;
    uint32_t incl = c;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      const uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
      if (lane >= o) incl += y;
    }
    if (lane == 31) wsum[w] = incl;
    __syncthreads();
    uint32_t off = 0, tot = 0;
#pragma unroll
    for (int k = 0; k < kPartThreads / 32; ++k) {
      off += k < w ? wsum[k] : 0u;
      tot += wsum[k];
    }
    if (i < width) {
      m.off[i] = run0 + off + incl - c;
      gb[i] = c ? atomicAdd(&cur[qb + i], c) : 0u;   // global base of the slot's range
      m.cnt[i] = 0;                                 // ranks taken: clean for the next tile
    }
    run0 += tot;
    __syncthreads();
  }
  if (t == 0) m.total = run0;
}

// Stage item (slot, rank) in the tile's partition-grouped order.
__device__ __forceinline__ void tile_stage(TileMap& m, uint32_t slot, uint32_t rank, uint4 rec) {
  const uint32_t i = m.off[slot] + rank;
  m.stage[i] = rec;
  m.sslot[i] = (uint16_t)slot;
}

// After a barrier: write the staged records; consecutive lanes write consecutive
// records of one partition (coalesced runs instead of one line per lane).
__device__ __forceinline__ void tile_flush(TileMap& m, uint32_t nitems, uint8_t* out, int rec_bytes) {
  for (uint32_t i = threadIdx.x; i < nitems; i += blockDim.x) {
    const uint32_t sl = m.sslot[i];
    *(uint4*)(out + (size_t)(m.cnt[sl] + (i - m.off[sl])) * rec_bytes) = m.stage[i];
  }
}

template <int NV>
__device__ __forceinline__ uint4 pack_rec16(uint64_t key, const int32_t (&v)[NV > 0 ? NV : 1]) {
  return make_uint4((uint32_t)key, (uint32_t)(key >> 32), NV > 0 ? (uint32_t)v[0] : 0u,
                    NV > 1 ? (uint32_t)v[NV > 1 ? 1 : 0] : 0u);
}

template <int NV>
__device__ __forceinline__ void store_rec(uint8_t* rec, uint64_t key, const int32_t (&v)[NV > 0 ? NV : 1]) {
  uint32_t z[8] = {(uint32_t)key, (uint32_t)(key >> 32), 0, 0, 0, 0, 0, 0};
#pragma unroll
  for (int i = 0; i < NV; ++i) z[2 + i] = (uint32_t)v[i];
  *(uint4*)rec = make_uint4(z[0], z[1], z[2], z[3]);
  if constexpr (NV > 2) *(uint4*)(rec + 16) = make_uint4(z[4], z[5], z[6], z[7]);
}

template <int NV>
__device__ __forceinline__ void load_rec(const uint8_t* rec, uint64_t& key, int32_t (&v)[NV > 0 ? NV : 1]) {
  const uint4 q0 = *(const uint4*)rec;
  key = (uint64_t)q0.x | ((uint64_t)q0.y << 32);
  uint32_t z[6] = {q0.z, q0.w, 0, 0, 0, 0};
  if constexpr (NV > 2) {
    const uint4 q1 = *(const uint4*)(rec + 16);
    z[2] = q1.x; z[3] = q1.y; z[4] = q1.z; z[5] = q1.w;
  }
#pragma unroll
  for (int i = 0; i < NV; ++i) v[i] = (int32_t)z[i];
}

// Level 1: rows -> records grouped by the top `pb` hash bits (cursors `cur`, output `out`).
template <class Sh, int NV>
__global__ void __launch_bounds__(kPartThreads, 2) k_part_scatter(const __grid_constant__ Plan p, PartArgs a, int pb,
                                                               uint32_t* cur, uint8_t* out) {
  extern __shared__ __align__(16) uint8_t dsm[];
  TileMap& map = *(TileMap*)dsm;
  __shared__ uint32_t wsum[32];
  const int64_t r0 = blockIdx.x * a.rows_per_blk;
  const int64_t r1 = min(p.n, r0 + a.rows_per_blk);
  const int lane = threadIdx.x & 31;
  // software pipeline: the next tile's rows are loaded before this tile's claims,
  // whose global atomics and barriers would otherwise serialise with the loads
  Row<Sh, NV, false> nx[kPartILP];
  bool nok[kPartILP];
  const int64_t woff = (int64_t)(threadIdx.x >> 5) * 128;
  if (r0 < r1) part_rows<Sh, NV>(p, r0 + woff, r1, lane, nx, nok);
  tile_map_init(map);
  __syncthreads();
  for (int64_t base = r0; base < r1; base += kPartILP * blockDim.x) {
    tile_map_reset(map);
    Row<Sh, NV, false> x[kPartILP];
    bool ok[kPartILP];
    uint32_t slot[kPartILP], rank[kPartILP];
    const int64_t wbase = base + woff;
#pragma unroll
    for (int k = 0; k < kPartILP; ++k) {
      x[k] = nx[k];
      ok[k] = nok[k];
    }
    if (base + kPartILP * blockDim.x < r1) part_rows<Sh, NV>(p, wbase + kPartILP * blockDim.x, r1, lane, nx, nok);
    __syncthreads();
#pragma unroll
    for (int k = 0; k < kPartILP; ++k) {
      if (x[k].q && !ok[k]) {               // exact per-row path straight into the HBM table
        uint8_t* e = table_find_or_insert(p.table, p.mask, p.stride, (uint64_t)x[k].key, p.status);
        if (e) update_entry_slow(p, e, part_row(wbase, lane, k));
        if ((uint64_t)x[k].key != ~0ULL) a.slowflag[part_of((uint64_t)x[k].key, a.pbits)] = 1u;   // region touched
      }
      if (ok[k]) tile_map_add(map, part_of((uint64_t)x[k].key, pb), slot[k], rank[k]);
    }
    __syncthreads();
    tile_map_claim(map, cur, wsum);
    __syncthreads();
#pragma unroll
    for (int k = 0; k < kPartILP; ++k) {
      if (!ok[k]) continue;
      int32_t v[NV > 0 ? NV : 1];
#pragma unroll
      for (int i = 0; i < NV; ++i) v[i] = (int32_t)x[k].vi[i];
      if constexpr (NV <= 2) tile_stage(map, slot[k], rank[k], pack_rec16<NV>((uint64_t)x[k].key, v));
      else store_rec<NV>(out + (size_t)(map.cnt[slot[k]] + rank[k]) * a.rec_bytes, (uint64_t)x[k].key, v);
    }
    __syncthreads();
    if constexpr (NV <= 2) {
      tile_flush(map, map.total, out, a.rec_bytes);
      __syncthreads();
    }
  }
}

// One level, no tiles: every qualifying row claims its record position with one returning
// atomic on its partition's cursor (lanes sharing lane 0's partition — hot keys — take one
// atomic of lane 0) and stores its 16-byte record there.  No barriers or shared-memory
// maps: the claims of kPartILP rows are in flight together, and the next rows' loads are
// issued before this group's claims return.  The P cursors keep one partially written
// line per partition open in L2 (P x 128 B = 2 MB at 2^14 partitions), so the scattered
// 16-byte stores still leave L2 as whole sectors.
// PF: the next rows' loads are issued before this group's claims (1 CTA / SM); otherwise
// RG groups of kPartILP rows per thread are loaded, then all their claims issued (2 CTAs / SM).
template <class Sh, int NV, bool PF, int RG>
__global__ void __launch_bounds__(kPartThreads, PF ? 1 : 2) k_part_scatter_direct(const __grid_constant__ Plan p, PartArgs a) {
  constexpr int R = kPartILP * RG;
  const int64_t r0 = blockIdx.x * a.rows_per_blk;
  const int64_t r1 = min(p.n, r0 + a.rows_per_blk);
  const int lane = threadIdx.x & 31;
  const uint32_t lt = lanemask_lt();
  const int64_t woff = (int64_t)(threadIdx.x >> 5) * 128;
  Row<Sh, NV, false> nx[PF ? kPartILP : 1];
  bool nok[PF ? kPartILP : 1];
  if constexpr (PF)
    if (r0 < r1) part_rows<Sh, NV>(p, r0 + woff, r1, lane, nx, nok);
  for (int64_t base0 = r0; base0 < r1; base0 += R * blockDim.x) {
    Row<Sh, NV, false> x[R];
    bool ok[R];
    const int64_t wbase0 = base0 + woff;
    if constexpr (PF) {
#pragma unroll
      for (int k = 0; k < kPartILP; ++k) {
        x[k] = nx[k];
        ok[k] = nok[k];
      }
      if (base0 + kPartILP * blockDim.x < r1) part_rows<Sh, NV>(p, wbase0 + kPartILP * blockDim.x, r1, lane, nx, nok);
    } else {
#pragma unroll
      for (int g = 0; g < RG; ++g) {
        Row<Sh, NV, false> y[kPartILP];
        bool yk[kPartILP];
        part_rows<Sh, NV>(p, wbase0 + (int64_t)g * kPartILP * blockDim.x, r1, lane, y, yk);
#pragma unroll
        for (int k = 0; k < kPartILP; ++k) {
          x[g * kPartILP + k] = y[k];
          ok[g * kPartILP + k] = yk[k];
        }
      }
    }
    uint32_t part[R], ret[R];
    unsigned same[R];
#pragma unroll
    for (int k = 0; k < R; ++k) {
      part[k] = ok[k] ? part_of((uint64_t)x[k].key, a.pbits) : 0xFFFFFFFFu;
      const uint32_t p0 = __shfl_sync(0xffffffffu, part[k], 0);
      same[k] = __ballot_sync(0xffffffffu, ok[k] && part[k] == p0);
      ret[k] = 0;
      if (ok[k] && (lane == 0 || part[k] != p0))
        ret[k] = atomicAdd(&a.curp[(size_t)part[k] << a.curp_shift], lane == 0 ? (uint32_t)__popc(same[k]) : 1u);
    }
#pragma unroll
    for (int k = 0; k < R; ++k) {
      const uint32_t b0 = __shfl_sync(0xffffffffu, ret[k], 0);
      if (x[k].q && !ok[k]) {               // exact per-row path straight into the HBM table
        uint8_t* e = table_find_or_insert(p.table, p.mask, p.stride, (uint64_t)x[k].key, p.status);
        if (e) update_entry_slow(p, e, part_row(wbase0 + (int64_t)(k / kPartILP) * kPartILP * blockDim.x, lane, k % kPartILP));
        if ((uint64_t)x[k].key != ~0ULL) a.slowflag[part_of((uint64_t)x[k].key, a.pbits)] = 1u;
      }
      if (!ok[k]) continue;
      const uint32_t pos = (same[k] >> lane) & 1u ? b0 + (uint32_t)__popc(same[k] & lt) : ret[k];
      int32_t v[NV > 0 ? NV : 1];
#pragma unroll
      for (int i = 0; i < NV; ++i) v[i] = (int32_t)x[k].vi[i];
      if constexpr (NV <= 2) *(uint4*)(a.recs + (size_t)pos * 16) = pack_rec16<NV>((uint64_t)x[k].key, v);
      else store_rec<NV>(a.recs + (size_t)pos * a.rec_bytes, (uint64_t)x[k].key, v);
    }
  }
}

// The same scatter as a three-stage software pipeline over tiles of kPartILP rows per
// thread: iteration i issues the loads of tile i + 1, the claims of tile i (whose rows
// arrived during iteration i - 1) and the record stores of tile i - 1 (whose claims were
// issued in iteration i - 1).  Every wait then covers one load and one claim latency: the
// one-stage kernel above was latency-bound (ncu: long-scoreboard stalls on the key loads
// and on the claim results, L2 at 37 % of its throughput, one CTA of 16 warps per SM).
// Records of NV <= 2 values only (16 bytes).
// One pipeline stage: tile `base` (rows x, arrived) claims into set C; set P (the previous
// tile's records and claims) is stored; the next tile's loads were issued by the caller.
// C and P alternate between two register sets (the loop is unrolled by two), so no claim
// result is moved between registers before it is used: a move would wait for it.
struct PipeSet {
  uint4 rec[kPartILP];
  uint32_t ret[kPartILP];
  unsigned same[kPartILP];
  bool ok[kPartILP];
};

template <class Sh, int NV>
__device__ __forceinline__ void pipe_stage(const Plan& p, const PartArgs& a, int64_t wbase, bool have,
                                           const Row<Sh, NV, false> (&x)[kPartILP], const bool (&xok)[kPartILP],
                                           PipeSet& C, const PipeSet& P, int lane, uint32_t lt) {
#pragma unroll
  for (int k = 0; k < kPartILP; ++k) {
    const bool ok = have && xok[k];
    const uint32_t part = ok ? part_of((uint64_t)x[k].key, a.pbits) : 0xFFFFFFFFu;
    const uint32_t p0 = __shfl_sync(0xffffffffu, part, 0);
    C.same[k] = __ballot_sync(0xffffffffu, ok && part == p0);
    C.ret[k] = 0;
    if (ok && (lane == 0 || part != p0))
      C.ret[k] = atomicAdd(&a.curp[(size_t)part << a.curp_shift], lane == 0 ? (uint32_t)__popc(C.same[k]) : 1u);
    C.ok[k] = ok;
    if (have && x[k].q && !ok) {           // exact per-row path straight into the HBM table
      uint8_t* e = table_find_or_insert(p.table, p.mask, p.stride, (uint64_t)x[k].key, p.status);
      if (e) update_entry_slow(p, e, part_row(wbase, lane, k));
      if ((uint64_t)x[k].key != ~0ULL) a.slowflag[part_of((uint64_t)x[k].key, a.pbits)] = 1u;
    }
    int32_t v[NV > 0 ? NV : 1];
#pragma unroll
    for (int i = 0; i < NV; ++i) v[i] = (int32_t)x[k].vi[i];
    C.rec[k] = pack_rec16<NV>((uint64_t)x[k].key, v);
  }
#pragma unroll
  for (int k = 0; k < kPartILP; ++k) {     // stores of the previous tile
    const uint32_t b0 = __shfl_sync(0xffffffffu, P.ret[k], 0);
    if (P.ok[k]) {
      const uint32_t pos = (P.same[k] >> lane) & 1u ? b0 + (uint32_t)__popc(P.same[k] & lt) : P.ret[k];
      *(uint4*)(a.recs + (size_t)pos * 16) = P.rec[k];
    }
  }
}

// The one-level scatter as a three-stage software pipeline over tiles of kPartILP rows per
// thread: a stage issues the loads of tile i + 1, the claims of tile i (whose rows arrived
// during stage i - 1) and the record stores of tile i - 1 (whose claims were issued in
// stage i - 1).  Every wait then covers one load and one claim latency: the one-stage kernel
// above is latency-bound (ncu: long-scoreboard stalls on the key loads and on the claim
// results, L2 at 37 % of its throughput, one CTA of 16 warps per SM).  16-byte records.
template <class Sh, int NV>
__global__ void __launch_bounds__(kPartThreads, 1) k_part_scatter_pipe(const __grid_constant__ Plan p, PartArgs a) {
  static_assert(NV <= 2, "16-byte records");
  const int64_t r0 = blockIdx.x * a.rows_per_blk;
  const int64_t r1 = min(p.n, r0 + a.rows_per_blk);
  const int lane = threadIdx.x & 31;
  const uint32_t lt = lanemask_lt();
  const int64_t woff = (int64_t)(threadIdx.x >> 5) * 128;
  const int64_t step = kPartILP * blockDim.x;
  Row<Sh, NV, false> xa[kPartILP], xb[kPartILP];
  bool oka[kPartILP], okb[kPartILP];
  PipeSet A, B;
#pragma unroll
  for (int k = 0; k < kPartILP; ++k) B.ok[k] = false;
  if (r0 < r1) part_rows<Sh, NV>(p, r0 + woff, r1, lane, xa, oka);
  // stage order per pair: (tile in xa -> A, stores B), (tile in xb -> B, stores A)
  for (int64_t base = r0; base < r1; base += 2 * step) {
    if (base + step < r1) part_rows<Sh, NV>(p, base + step + woff, r1, lane, xb, okb);
    pipe_stage<Sh, NV>(p, a, base + woff, true, xa, oka, A, B, lane, lt);
    const bool h1 = base + step < r1;
    if (base + 2 * step < r1) part_rows<Sh, NV>(p, base + 2 * step + woff, r1, lane, xa, oka);
    pipe_stage<Sh, NV>(p, a, base + step + woff, h1, xb, okb, B, A, lane, lt);
  }
  // drain: the last stage claimed into B (a pair always ends with B)
#pragma unroll
  for (int k = 0; k < kPartILP; ++k) {
    const uint32_t b0 = __shfl_sync(0xffffffffu, B.ret[k], 0);
    if (B.ok[k]) {
      const uint32_t pos = (B.same[k] >> lane) & 1u ? b0 + (uint32_t)__popc(B.same[k] & lt) : B.ret[k];
      *(uint4*)(a.recs + (size_t)pos * 16) = B.rec[k];
    }
  }
}

__global__ void k_part_cur_pad(const uint32_t* offs, uint32_t* curp, int shift, int64_t L) {
  const int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x;
  if (i < L) curp[i << shift] = offs[i];
}

// Lazily zeroed HBM table (PartArgs::lazy): only the regions that will hold entries are
// cleared — partitions with exact-path rows (slowflag, set by the count pass) and
// partitions split over several pass-2 work items.  One CTA per partition.
__global__ void k_part_zero_regions(const __grid_constant__ Plan p, PartArgs a) {
  const int64_t q = blockIdx.x;
  const int64_t m = *a.m_dev;
  const int64_t n = (q + 1 >= (1LL << a.pbits) ? m : (int64_t)a.offs[q + 1]) - (int64_t)a.offs[q];
  if (!a.slowflag[q] && n <= kPartItem) return;             // CTA-uniform
  uint4* r = (uint4*)(p.table + ((size_t)q << kPartCapBits) * p.stride);
  const int nq = (int)(((size_t)p.stride << kPartCapBits) / 16);
  for (int i = threadIdx.x; i < nq; i += blockDim.x) r[i] = make_uint4(0, 0, 0, 0);
}

// Level 1 with per-block ranges: rows -> records grouped by the top b1 hash bits (2^b1 <=
// 256 partitions).  The count pass left each row block's level-1 counts and their scan
// (a.cnt1: block c's range in level-1 partition t starts at cnt1[t][c]), so the block
// advances its own cursors in shared memory: no global claims, and a block keeps only
// 2^b1 partially written lines open in L2.  Per tile: ranks by shared atomics on the
// 2^b1 counters, one scan, records staged in partition order and written as runs.
// The level-1 tile state of a T-thread block (~21 KB at T = 256: four blocks of 8 warps per
// SM, so one block's barriers overlap the others' loads; at T = 512 two blocks fit).
template <int T>
struct L1Map {
  uint4 stage[kPartILP * T];              // the tile's records, grouped by partition
  uint32_t cnt[256];                      // ranks, then zero again
  uint32_t off[256];                      // the slot's first index in the staging area
  uint32_t key[256];                      // block cursor
  uint32_t gb[256];                       // this tile's global base per slot
  uint8_t sslot[kPartILP * T];            // slot of each staged record
  uint32_t total;
};

template <class Sh, int NV, int T, bool SPARSE>
__global__ void __launch_bounds__(T, T == 256 ? 4 : 2) k_part_scatter_l1(const __grid_constant__ Plan p, PartArgs a,
                                                                         uint8_t* out) {
  if (a.sparse_dev && (*a.sparse_dev != 0) != SPARSE) return;     // the other variant runs (grid-uniform)
  extern __shared__ __align__(16) uint8_t dsm[];
  L1Map<T>& m = *(L1Map<T>*)dsm;
  uint32_t* gb = m.gb;
  __shared__ uint32_t wsum[32];
  const int P1 = 1 << a.b1;
  const int64_t r0 = blockIdx.x * a.rows_per_blk;
  const int64_t r1 = min(p.n, r0 + a.rows_per_blk);
  const int lane = threadIdx.x & 31, t = threadIdx.x, w = t >> 5;
  for (int i = t; i < P1; i += blockDim.x) {
    m.cnt[i] = 0;
    m.key[i] = a.cnt1[(size_t)i * a.nblk + blockIdx.x];
  }
  Row<Sh, NV, false> nx[kPartILP];
  bool nok[kPartILP];
  const int64_t woff = (int64_t)(threadIdx.x >> 5) * 128;
  // sparse mode: the block's list of qualifying rows (count pass) is the row source
  constexpr bool sparse = SPARSE;
  const int64_t s1 = sparse ? r0 + (int64_t)a.nq[blockIdx.x] : r1;
  if (!sparse && r0 < r1) part_rows<Sh, NV>(p, r0 + woff, r1, lane, nx, nok);
  __syncthreads();
  for (int64_t base = r0; base < s1; base += kPartILP * blockDim.x) {
    Row<Sh, NV, false> x[kPartILP];
    bool ok[kPartILP];
    int64_t rid[kPartILP];
    uint32_t q[kPartILP], rank[kPartILP];
    const int64_t wbase = base + woff;
    if constexpr (SPARSE) {
#pragma unroll
      for (int k = 0; k < kPartILP; ++k) {
        const int64_t j = base + (int64_t)k * blockDim.x + threadIdx.x;
        rid[k] = j < s1 ? (int64_t)a.soids[j] : p.n;
      }
#pragma unroll
      for (int k = 0; k < kPartILP; ++k) {
        eval_one<Sh, NV, false>(p, rid[k], x[k]);       // (row n: x.q = false)
        ok[k] = x[k].q && x[k].fast && !Sh::special(x[k].key);
      }
    } else {
#pragma unroll
      for (int k = 0; k < kPartILP; ++k) {
        x[k] = nx[k];
        ok[k] = nok[k];
        rid[k] = part_row(wbase, lane, k);
      }
      if (base + kPartILP * blockDim.x < r1) part_rows<Sh, NV>(p, wbase + kPartILP * blockDim.x, r1, lane, nx, nok);
    }
#pragma unroll
    for (int k = 0; k < kPartILP; ++k) {
      if (x[k].q && !ok[k]) {               // exact per-row path straight into the HBM table
        uint8_t* e = table_find_or_insert(p.table, p.mask, p.stride, (uint64_t)x[k].key, p.status);
        if (e) update_entry_slow(p, e, rid[k]);
        if ((uint64_t)x[k].key != ~0ULL) a.slowflag[part_of((uint64_t)x[k].key, a.pbits)] = 1u;
      }
      q[k] = ok[k] ? part_of((uint64_t)x[k].key, a.b1) : 0u;
      if (ok[k]) rank[k] = atomicAdd(&m.cnt[q[k]], 1u);
    }
    __syncthreads();
    // offsets in the staging area (exclusive scan of the <= 256 counts) and global bases
    {
      const uint32_t c = t < P1 ? m.cnt[t] : 0u;
      uint32_t incl = c;
#pragma unroll
      for (int o = 1; o < 32; o <<= 1) {
        const uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
        if (lane >= o) incl += y;
      }
      if (lane == 31 && w < 8) wsum[w] = incl;
      __syncthreads();
      if (t < P1) {
        uint32_t off = 0;
        for (int k = 0; k < w; ++k) off += wsum[k];
        m.off[t] = off + incl - c;
        const uint32_t g = m.key[t];
        m.key[t] = g + c;                    // block cursor
        gb[t] = g;                           // this tile's global base
        m.cnt[t] = 0;                        // ranks taken: ready for the next tile (its atomics
                                             // follow two more barriers)
        if (t == P1 - 1) m.total = off + incl;
      }
    }
    __syncthreads();
#pragma unroll
    for (int k = 0; k < kPartILP; ++k) {
      if (!ok[k]) continue;
      int32_t v[NV > 0 ? NV : 1];
#pragma unroll
      for (int i = 0; i < NV; ++i) v[i] = (int32_t)x[k].vi[i];
      if constexpr (NV <= 2) {
        const uint32_t i = m.off[q[k]] + rank[k];
        m.stage[i] = pack_rec16<NV>((uint64_t)x[k].key, v);
        m.sslot[i] = (uint8_t)q[k];
      }
      else store_rec<NV>(out + (size_t)(gb[q[k]] + rank[k]) * a.rec_bytes, (uint64_t)x[k].key, v);
    }
    __syncthreads();
    if constexpr (NV <= 2)
      for (uint32_t i = t; i < m.total; i += blockDim.x) {
        const uint32_t sl = m.sslot[i];
        *(uint4*)(out + (size_t)(gb[sl] + (i - m.off[sl])) * 16) = m.stage[i];
      }
    __syncthreads();                      // stage / gb / off are rewritten by the next tile
  }
}

// Level 2: records grouped by their top b1 hash bits -> records grouped by all pbits.
// A tile of consecutive level-1 records spans one or two level-1 partitions, so it
// meets at most ~2^(pbits-b1) final partitions: the tile claims aggregate again.
template <int NV>
__global__ void __launch_bounds__(kPartThreads, 2) k_part_scatter2(PartArgs a) {
  extern __shared__ __align__(16) uint8_t dsm[];
  TileMap& map = *(TileMap*)dsm;
  __shared__ uint32_t wsum[32];
  uint32_t* gb = map.off + kTileMap / 2;  // direct-map tiles: global bases (slots < kDirectMap)
  static_assert(kDirectMap <= kTileMap / 2, "direct-map bases share the off array");
  const int64_t m = *a.m_dev;
  constexpr int TILE = kPartILP * kPartThreads;
  const int64_t per = ((m + gridDim.x - 1) / gridDim.x + TILE - 1) / TILE * TILE;
  const int64_t j0 = blockIdx.x * per, j1 = min(m, j0 + per);
  uint64_t nkey[kPartILP];
  int32_t nv[kPartILP][NV > 0 ? NV : 1];
  auto fetch = [&](int64_t b) {
#pragma unroll
    for (int k = 0; k < kPartILP; ++k) {
      const int64_t j = b + k * kPartThreads + threadIdx.x;
      if (j < j1) load_rec<NV>(a.tmp + (size_t)j * a.rec_bytes, nkey[k], nv[k]);
    }
  };
  if (j0 < j1) fetch(j0);
  tile_map_init(map);
  __syncthreads();
  bool hashed = false;                    // the previous tile used the hashed map (CTA-uniform)
  for (int64_t base = j0; base < j1; base += TILE) {
    if (hashed || NV > 2) {
      tile_map_reset(map);
      __syncthreads();
    }
    uint64_t key[kPartILP];
    int32_t v[kPartILP][NV > 0 ? NV : 1];
    bool ok[kPartILP];
    uint32_t slot[kPartILP], rank[kPartILP];
#pragma unroll
    for (int k = 0; k < kPartILP; ++k) {
      ok[k] = base + k * kPartThreads + threadIdx.x < j1;
      key[k] = nkey[k];
#pragma unroll
      for (int i = 0; i < NV; ++i) v[k][i] = nv[k][i];
    }
    if (base + TILE < j1) fetch(base + TILE);
    // the tile's final partitions lie in [qb, qb + width): its first and last record's
    // level-1 partitions bound them (level-1 records are in level-1 order)
    const int sh = a.pbits - a.b1;
    const uint32_t q1f = part_of(*(const uint64_t*)(a.tmp + (size_t)base * a.rec_bytes), a.b1);
    const uint32_t q1l = part_of(*(const uint64_t*)(a.tmp + (size_t)(min(base + TILE, j1) - 1) * a.rec_bytes), a.b1);
    const uint32_t qb = q1f << sh, width = (q1l - q1f + 1) << sh;
    const bool dmap = a.b1 > 0 && width <= kDirectMap && NV <= 2;   // CTA-uniform
    hashed = !dmap;
    if (dmap) {                           // direct-indexed map: no hashing, no key slots
#pragma unroll
      for (int k = 0; k < kPartILP; ++k)
        if (ok[k]) {
          slot[k] = part_of(key[k], a.pbits) - qb;
          rank[k] = atomicAdd(&map.cnt[slot[k]], 1u);
        }
      __syncthreads();
      tile_dmap_claim(map, width, qb, a.cur, wsum, gb);
      __syncthreads();
#pragma unroll
      for (int k = 0; k < kPartILP; ++k)
        if (ok[k]) tile_stage(map, slot[k], rank[k], pack_rec16<NV>(key[k], v[k]));
      __syncthreads();
      for (uint32_t i = threadIdx.x; i < map.total; i += blockDim.x) {
        const uint32_t sl = map.sslot[i];
        *(uint4*)(a.recs + (size_t)(gb[sl] + (i - map.off[sl])) * 16) = map.stage[i];
      }
      __syncthreads();                    // stage / off / gb are rewritten by the next tile
      continue;
    }
#pragma unroll
    for (int k = 0; k < kPartILP; ++k)
      if (ok[k]) tile_map_add(map, part_of(key[k], a.pbits), slot[k], rank[k]);
    __syncthreads();
    tile_map_claim(map, a.cur, wsum);
    __syncthreads();
#pragma unroll
    for (int k = 0; k < kPartILP; ++k) {
      if (!ok[k]) continue;
      if constexpr (NV <= 2) tile_stage(map, slot[k], rank[k], pack_rec16<NV>(key[k], v[k]));
      else store_rec<NV>(a.recs + (size_t)(map.cnt[slot[k]] + rank[k]) * a.rec_bytes, key[k], v[k]);
    }
    __syncthreads();
    if constexpr (NV <= 2) {
      tile_flush(map, map.total, a.recs, a.rec_bytes);
      __syncthreads();
    }
  }
}

// cursors of level 1: start of level-1 partition q1 = start of final partition q1 << b2
__global__ void k_part_cur1(const uint32_t* offs, uint32_t* cur1, int b1, int b2) {
  const int i = blockIdx.x * blockDim.x + threadIdx.x;
  if (i < (1 << b1)) cur1[i] = offs[(size_t)i << b2];
}

// ------------------------------------------------------------------ scan (exclusive, u32)
__global__ void __launch_bounds__(kScanThreads) k_scan_chunks(const uint32_t* in, uint32_t* out, uint32_t* sums,
                                                               int64_t n) {
  __shared__ uint32_t wsum[kScanThreads / 32];
  const int64_t c0 = (int64_t)blockIdx.x * kScanChunk + (int64_t)threadIdx.x * kScanPer;
  uint32_t v[kScanPer], t = 0;
#pragma unroll
  for (int i = 0; i < kScanPer; ++i) {
    v[i] = c0 + i < n ? in[c0 + i] : 0u;
    t += v[i];
  }
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  uint32_t incl = t;
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    const uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
    if (lane >= o) incl += y;
  }
  if (lane == 31) wsum[w] = incl;
  __syncthreads();
  if (w == 0) {
    uint32_t s = wsum[lane];
    uint32_t si = s;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      const uint32_t y = __shfl_up_sync(0xffffffffu, si, o);
      if (lane >= o) si += y;
    }
    wsum[lane] = si - s;
    if (lane == 31) sums[blockIdx.x] = si;
  }
  __syncthreads();
  uint32_t run = wsum[w] + incl - t;
#pragma unroll
  for (int i = 0; i < kScanPer; ++i) {
    if (c0 + i < n) out[c0 + i] = run;
    run += v[i];
  }
}

// One CTA: exclusive scan of the chunk sums in place; total -> *total.
__global__ void __launch_bounds__(kScanThreads) k_scan_sums(uint32_t* sums, int64_t nchunks, int64_t* total) {
  __shared__ uint32_t wsum[kScanThreads / 32];
  __shared__ uint32_t carry;
  if (threadIdx.x == 0) carry = 0;
  __syncthreads();
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  for (int64_t base = 0; base < nchunks; base += kScanThreads) {
    const int64_t i = base + threadIdx.x;
    const uint32_t v = i < nchunks ? sums[i] : 0u;
    uint32_t incl = v;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      const uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
      if (lane >= o) incl += y;
    }
    if (lane == 31) wsum[w] = incl;
    __syncthreads();
    if (w == 0) {
      uint32_t s = wsum[lane], si = s;
#pragma unroll
      for (int o = 1; o < 32; o <<= 1) {
        const uint32_t y = __shfl_up_sync(0xffffffffu, si, o);
        if (lane >= o) si += y;
      }
      wsum[lane] = si - s;
    }
    __syncthreads();
    const uint32_t c = carry;
    if (i < nchunks) sums[i] = c + wsum[w] + incl - v;
    __syncthreads();
    if (threadIdx.x == kScanThreads - 1) carry = c + wsum[w] + incl;
    __syncthreads();
  }
  if (threadIdx.x == 0) *total = (int64_t)carry;
}

__global__ void k_scan_add(uint32_t* out, uint32_t* cur, const uint32_t* sums, int64_t n) {
  const int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x;
  if (i < n) cur[i] = out[i] += sums[i / kScanChunk];
}

// ------------------------------------------------------------------ pass 2: aggregate
// Exact HBM update of one record that the shared table could not take.
__device__ __forceinline__ void update_entry_rec(const Plan& p, uint8_t* e, const int32_t* v, int nv) {
  atomicAdd((unsigned long long*)(e + 8), 1ULL);
  for (int i = 0; i < nv; ++i) {
    const DevValue& d = p.vals[i];
    const int64_t x = v[i];
    if (d.off_sum >= 0) atomic_add_i128((uint64_t*)(e + d.off_sum), (uint64_t)x, (uint64_t)(x >> 63));
    if (d.off_min >= 0) atomicMax((unsigned long long*)(e + d.off_min), (unsigned long long)enc_min_i(x));
    if (d.off_max >= 0) atomicMax((unsigned long long*)(e + d.off_max), (unsigned long long)enc_max_i(x));
  }
}

// ---- the pass-2 shared table, field-major: keys u64[kPartCap] (~key, 0 = empty), then one
// u32[kPartCap] array per 4-byte field of the CTA-table entry layout the planner assigned
// (count at entry offset 8, per value sum lo / hi, MIN, MAX at d.co_*): entry offset co ->
// array (co - 8) / 4.  Lanes of an atomic instruction on different slots then hit different
// banks (an AoS entry of 32 bytes put every entry's count field in 4 of the 32 banks:
// ~16 wavefronts per atomic instruction on C3).  SUM: the biased sum of (x + 2^31) as a
// 64-bit {lo, hi} pair; lo is added atomically and the carry out of it (seen in the value
// the atomic returns) is added to hi, so one atomic per row (exact: sum = biased - count * 2^31).
__device__ __forceinline__ int32_t dec32_max(uint32_t e) { return (int32_t)(e ^ 0x80000000u); }
__device__ __forceinline__ int32_t dec32_min(uint32_t e) { return dec32_max(~e); }
__device__ __forceinline__ uint64_t* pkey(uint8_t* tab, int slot) { return (uint64_t*)tab + slot; }
__device__ __forceinline__ uint32_t* pf32(uint8_t* tab, int slot, int co) {
  return (uint32_t*)(tab + 8 * (size_t)kPartCap + (size_t)kPartCap * (co - 8)) + slot;
}
__device__ __forceinline__ const uint32_t* pf32(const uint8_t* tab, int slot, int co) {
  return (const uint32_t*)(tab + 8 * (size_t)kPartCap + (size_t)kPartCap * (co - 8)) + slot;
}
__device__ __forceinline__ int64_t part_sum(const uint8_t* tab, int slot, int co_lo, uint32_t cnt) {
  const uint64_t b = (uint64_t)*pf32(tab, slot, co_lo) | ((uint64_t)*pf32(tab, slot, co_lo + 4) << 32);
  return (int64_t)(b - ((uint64_t)cnt << 31));
}
__device__ __forceinline__ void part_add_sum(uint8_t* tab, int slot, int co_lo, uint64_t biased) {
  const uint32_t a = (uint32_t)biased, hi = (uint32_t)(biased >> 32);
  const uint32_t old = atomicAdd(pf32(tab, slot, co_lo), a);
  const uint32_t c = hi + (uint32_t)(old + a < old);
  if (c) atomicAdd(pf32(tab, slot, co_lo + 4), c);
}

// Field offsets of value i: from the plan, or (FIX: one value with SUM, MIN and MAX — the
// C3 / C5 plans) the compile-time layout co_lo 12, co_hi 16, co_min 20, co_max 24, which
// removes the per-record constant-bank loads and flag branches.
template <bool FIX>
__device__ __forceinline__ void part_cos(const Plan& p, int i, int& lo, int& mn, int& mx) {
  if constexpr (FIX) {
    lo = 12;
    mn = 20;
    mx = 24;
  } else {
    lo = p.vals[i].co_lo;
    mn = p.vals[i].co_min;
    mx = p.vals[i].co_max;
  }
}

// MIN / MAX field update; mmc: read first and skip the atomic when the value cannot improve
// (the field only grows, so a stale read can only cause an unneeded atomic).
__device__ __forceinline__ void part_max(uint32_t* f, uint32_t x, bool mmc) {
  if (!mmc || *(volatile uint32_t*)f < x) atomicMax(f, x);
}

// One record into slot `slot`.
template <int NV, bool FIX>
__device__ __forceinline__ void part_add(const Plan& p, uint8_t* tab, int slot, const int32_t (&v)[NV > 0 ? NV : 1],
                                         bool mmc) {
  atomicAdd(pf32(tab, slot, 8), 1u);
#pragma unroll
  for (int i = 0; i < NV; ++i) {
    if (!FIX && i >= p.nvals) break;
    int lo, mn, mx;
    part_cos<FIX>(p, i, lo, mn, mx);
    if (lo >= 0) part_add_sum(tab, slot, lo, (uint64_t)((uint32_t)v[i] ^ 0x80000000u));
    if (mn >= 0) part_max(pf32(tab, slot, mn), enc32_min(v[i]), mmc);
    if (mx >= 0) part_max(pf32(tab, slot, mx), enc32_max(v[i]), mmc);
  }
}

// A whole warp of records with the same key (heavy hitters): one combined update.
template <int NV, bool FIX>
__device__ __forceinline__ void part_add_warp(const Plan& p, uint8_t* tab, int slot, const int32_t (&v)[NV > 0 ? NV : 1],
                                              int lane) {
  if (lane == 0) atomicAdd(pf32(tab, slot, 8), 32u);
#pragma unroll
  for (int i = 0; i < NV; ++i) {
    if (!FIX && i >= p.nvals) break;
    int clo, cmn, cmx;
    part_cos<FIX>(p, i, clo, cmn, cmx);
    const uint32_t b = (uint32_t)v[i] ^ 0x80000000u;
    const uint32_t lo = __reduce_add_sync(0xffffffffu, b & 0xFFFFu);
    const uint32_t hi = __reduce_add_sync(0xffffffffu, b >> 16);
    const int32_t mn = __reduce_min_sync(0xffffffffu, v[i]);
    const int32_t mx = __reduce_max_sync(0xffffffffu, v[i]);
    if (lane == 0) {
      if (clo >= 0) part_add_sum(tab, slot, clo, (uint64_t)lo + ((uint64_t)hi << 16));
      if (cmn >= 0) atomicMax(pf32(tab, slot, cmn), enc32_min(mn));
      if (cmx >= 0) atomicMax(pf32(tab, slot, cmx), enc32_max(mx));
    }
  }
}

__device__ __forceinline__ int64_t part_start(const PartArgs& a, int64_t q, int64_t m) {
  return q >= (1LL << a.pbits) ? m : (int64_t)a.offs[q];
}

// Work items of pass 2: partition q is cut into ceil(n_q / kPartItem) items.
__global__ void k_part_items(PartArgs a) {
  const int64_t q = blockIdx.x * (int64_t)blockDim.x + threadIdx.x;
  if (q >= (1LL << a.pbits)) return;
  const int64_t m = *a.m_dev;
  const int64_t n = part_start(a, q + 1, m) - part_start(a, q, m);
  a.icnt[q] = (uint32_t)((n + kPartItem - 1) / kPartItem);
}

// Merge shared slot `slot` into the HBM table (atomics: other CTAs share the partition).
__device__ __forceinline__ void part_flush_slot(const Plan& p, const uint8_t* tab, int slot) {
  const uint64_t sk = *pkey((uint8_t*)tab, slot);
  const uint32_t cnt = *pf32(tab, slot, 8);
  if (sk == 0 || cnt == 0) return;
  uint8_t* e = table_find_or_insert(p.table, p.mask, p.stride, ~sk, p.status);
  if (!e) return;
  atomicAdd((unsigned long long*)(e + 8), (unsigned long long)cnt);
  for (int v = 0; v < p.nvals; ++v) {
    const DevValue& d = p.vals[v];
    if (d.co_lo >= 0) {
      const int64_t sum = part_sum(tab, slot, d.co_lo, cnt);
      atomic_add_i128((uint64_t*)(e + d.off_sum), (uint64_t)sum, (uint64_t)(sum >> 63));
    }
    if (d.co_min >= 0)
      atomicMax((unsigned long long*)(e + d.off_min), (unsigned long long)enc_min_i(dec32_min(*pf32(tab, slot, d.co_min))));
    if (d.co_max >= 0)
      atomicMax((unsigned long long*)(e + d.off_max), (unsigned long long)enc_max_i(dec32_max(*pf32(tab, slot, d.co_max))));
  }
}

// Merge a shared slot into the HBM table when this CTA is the only one aggregating its
// partition (a one-item partition): plain read-modify-write of the entry's fields — no
// other thread updates them (the scatter's exact path and this CTA's own overflow updates
// happened before the barrier).  The slot is still claimed with atomicCAS: linear probing
// may run into a neighbour partition's range.
__device__ __forceinline__ void part_flush_slot_excl(const Plan& p, const uint8_t* tab, int slot) {
  const uint64_t sk = *pkey((uint8_t*)tab, slot);
  const uint32_t cnt = *pf32(tab, slot, 8);
  if (sk == 0 || cnt == 0) return;
  uint8_t* e = table_find_or_insert(p.table, p.mask, p.stride, ~sk, p.status);
  if (!e) return;
  *(uint64_t*)(e + 8) += cnt;
  for (int v = 0; v < p.nvals; ++v) {
    const DevValue& d = p.vals[v];
    if (d.co_lo >= 0) {
      I128 x{*(const uint64_t*)(e + d.off_sum), *(const uint64_t*)(e + d.off_sum + 8)};
      x = i128_add(x, i128_from_i64(part_sum(tab, slot, d.co_lo, cnt)));
      *(uint64_t*)(e + d.off_sum) = x.lo;
      *(uint64_t*)(e + d.off_sum + 8) = x.hi;
    }
    if (d.co_min >= 0) {
      uint64_t* f = (uint64_t*)(e + d.off_min);
      *f = max(*f, enc_min_i(dec32_min(*pf32(tab, slot, d.co_min))));
    }
    if (d.co_max >= 0) {
      uint64_t* f = (uint64_t*)(e + d.off_max);
      *f = max(*f, enc_max_i(dec32_max(*pf32(tab, slot, d.co_max))));
    }
  }
}

// Shared-table find-or-insert for pass 2 -> slot, or -1 (probe limit).  Triangular
// (quadratic) probing from the home slot: linear probing's clusters made the warp-wide
// longest probe sequence the cost of every lookup at load 1/2 (ncu on C5 with 2^16 groups:
// ~half of pass 2's instructions in the probe loop).  The shared table's layout is private to
// the CTA (entries reach HBM through table_find_or_insert or as output rows).
constexpr int kPartProbes = 64;

// Home slot in the pass-2 shared table: multiplicative (Fibonacci) hashing — the partition
// already fixed the key's top fmix64 bits, and the shared layout is private to the CTA, so
// one 64-bit multiply replaces a second fmix64 per record.
__device__ __forceinline__ uint32_t part_home(uint64_t key) {
  return (uint32_t)((key * 0x9E3779B97F4A7C15ULL) >> (64 - kPartCapBits));
}

__device__ __forceinline__ int part_find(uint8_t* tab, uint64_t key, bool direct, int pbits) {
  const uint64_t sk = ~key;
  (void)direct;
  (void)pbits;
  uint32_t i = part_home(key);
  for (int probe = 0; probe < kPartProbes; ++probe) {
    uint64_t* kp = pkey(tab, (int)i);
    const uint64_t cur = *(volatile uint64_t*)kp;
    if (cur == sk) return (int)i;
    if (cur == 0) {
      const uint64_t prev = atomicCAS((unsigned long long*)kp, 0ULL, (unsigned long long)sk);
      if (prev == 0 || prev == sk) return (int)i;
    }
    i = (i + probe + 1) & (kPartCap - 1);   // triangular (quadratic) probing
  }
  return -1;
}

// Claim path of part_find_warp, out of line: the same probe sequence with CAS from slot i
// (the first empty slot this lane saw, reached after `np` steps).
static __device__ __noinline__ int part_claim_slow(uint8_t* tab, uint64_t key, uint32_t i, int np) {
  const uint64_t sk = ~key;
  for (int probe = np; probe < kPartProbes; ++probe) {
    uint64_t* kp = pkey(tab, (int)i);
    const uint64_t cur = *(volatile uint64_t*)kp;
    if (cur == sk) return (int)i;
    if (cur == 0) {
      const uint64_t prev = atomicCAS((unsigned long long*)kp, 0ULL, (unsigned long long)sk);
      if (prev == 0 || prev == sk) return (int)i;
    }
    i = (i + probe + 1) & (kPartCap - 1);
  }
  return -1;
}

// part_find for a whole warp (every lane calls it; `act` = the lane has a record): the home
// slot is read by every lane at once and a key found there costs no branch; lanes still
// searching probe in a warp-uniform loop, and claims (a key new to the table) go out of
// line.  The per-lane probe loop of part_find ran at ~13 active lanes per warp on C5 with
// 2^16 groups (ncu: Avg. Active Threads Per Warp 13.07): every warp paid its longest probe
// sequence and its CAS branch structure.  Same slots, same probe limit as part_find.
__device__ __forceinline__ int part_find_warp(uint8_t* tab, uint64_t key, bool act, bool direct, int pbits) {
  const uint64_t sk = ~key;
  (void)direct;
  (void)pbits;
  uint32_t i = part_home(key);
  uint64_t c = *(volatile uint64_t*)pkey(tab, (int)i);
  int ts = act && c == sk ? (int)i : -1;
  if (__any_sync(0xffffffffu, act && ts < 0)) {
    bool pend = act && ts < 0 && c != 0;
    bool claim = act && ts < 0 && c == 0;
    int np = 0;                           // probe steps taken (slot i = home + np (np + 1) / 2)
    while (__any_sync(0xffffffffu, pend)) {
      if (pend) {
        i = (i + np + 1) & (kPartCap - 1);
        ++np;
        c = *(volatile uint64_t*)pkey(tab, (int)i);
        if (c == sk) {
          ts = (int)i;
          pend = false;
        } else if (c == 0) {
          claim = true;
          pend = false;
        } else if (np >= kPartProbes) {
          pend = false;                   // probe limit: overflow
        }
      }
    }
    if (__any_sync(0xffffffffu, claim))
      if (claim) ts = part_claim_slow(tab, key, i, np);
  }
  return ts;
}

// A shared slot as a table-format entry at e (partial output rows).
__device__ __forceinline__ void part_store_slot(const Plan& p, const uint8_t* tab, int slot, uint8_t* e) {
  const uint64_t sk = *pkey((uint8_t*)tab, slot);
  const uint32_t cnt = *pf32(tab, slot, 8);
  if (sk == 0 || cnt == 0) return;
  *(uint64_t*)e = sk;
  *(uint64_t*)(e + 8) = cnt;
  for (int v = 0; v < p.nvals; ++v) {
    const DevValue& d = p.vals[v];
    if (d.co_lo >= 0) {
      const int64_t sum = part_sum(tab, slot, d.co_lo, cnt);
      *(uint64_t*)(e + d.off_sum) = (uint64_t)sum;
      *(uint64_t*)(e + d.off_sum + 8) = (uint64_t)(sum >> 63);
    }
    if (d.co_min >= 0) *(uint64_t*)(e + d.off_min) = enc_min_i(dec32_min(*pf32(tab, slot, d.co_min)));
    if (d.co_max >= 0) *(uint64_t*)(e + d.off_max) = enc_max_i(dec32_max(*pf32(tab, slot, d.co_max)));
  }
}

// One output row from a shared slot: final values or a partial row in the
// table-entry layout.
__device__ __forceinline__ void part_emit_row(const Plan& p, const PartArgs& a, const EmitArgs& ea, const uint8_t* tab,
                                              int slot, int64_t g) {
  const uint64_t key = ~*pkey((uint8_t*)tab, slot);
  const uint32_t cnt = *pf32(tab, slot, 8);
  if (ea.kind != EMIT_FINAL) {
    if (g >= ea.out_capacity) return;
    uint8_t* row = ea.partial_out + g * (int64_t)p.stride;
    part_store_slot(p, tab, slot, row);
    *(uint64_t*)row = key;
    return;
  }
  const FinPlan& f = ea.fin;
  if (g >= f.out_capacity) return;
  if (f.keys_out) f.keys_out[g] = (int64_t)key;
  for (int i = 0; i < a.npo; ++i) {
    const int kind = a.po[i].kind, f0 = a.po[i].f0;
    void* out = a.po[i].out;
    if (kind == 0) {
      ((int64_t*)out)[g] = cnt;
    } else if (kind <= 2) {
      const int64_t sum = part_sum(tab, slot, f0, cnt);
      if (kind == 1) ((ulonglong2*)out)[g] = make_ulonglong2((uint64_t)sum, (uint64_t)(sum >> 63));
      else ((double*)out)[g] = __ddiv_rn(__ll2double_rn(sum), __ull2double_rn(cnt));
    } else if (kind == 3) {
      ((int64_t*)out)[g] = dec32_min(*pf32(tab, slot, f0));
    } else {
      ((int64_t*)out)[g] = dec32_max(*pf32(tab, slot, f0));
    }
  }
}

#ifndef OCL_AGG_BLOCKS
#define OCL_AGG_BLOCKS 3
#endif
constexpr int kAggBlocks = OCL_AGG_BLOCKS;     // CTAs per SM of pass 2 (shared table 64 KB each)
#ifndef OCL_AGG_ILP
#define OCL_AGG_ILP 4
#endif
constexpr int kAggILP = OCL_AGG_ILP;           // records per thread in flight in pass 2

template <int NV, bool FIX>
__global__ void __launch_bounds__(kPartThreads, kAggBlocks) k_part_agg(const __grid_constant__ Plan p, PartArgs a,
                                                              const __grid_constant__ EmitArgs ea) {
  extern __shared__ __align__(16) uint8_t tab[];
  __shared__ int overflowed;
  __shared__ uint32_t wsum[kPartThreads / 32];
  __shared__ unsigned long long base_s;
  __shared__ uint16_t slot_list[kPartCap];
  const int lane = threadIdx.x & 31;
  const int64_t m = *a.m_dev;
  const int64_t nitems = *a.nitems_dev;
  const int64_t P = 1LL << a.pbits;
  const int cs = p.cta_stride;
  for (int64_t item = blockIdx.x; item < nitems; item += gridDim.x) {
    // the partition of this item: the largest q with ioff[q] <= item (= item when no
    // partition is split into several items)
    int64_t lo = nitems == P ? item : 0, hi = nitems == P ? item : P - 1;
    while (lo < hi) {
      const int64_t mid = (lo + hi + 1) >> 1;
      if ((int64_t)a.ioff[mid] <= item) lo = mid;
      else hi = mid - 1;
    }
    const int64_t q0 = part_start(a, lo, m), q1 = part_start(a, lo + 1, m);
    const int64_t s = q0 + (item - (int64_t)a.ioff[lo]) * kPartItem;
    const int64_t seg_end = min(q1, s + kPartItem);
    const bool exclusive = q1 - q0 <= kPartItem;
    // direct: rows emitted straight from shared memory (one-item partition, no exact-path rows)
    const bool direct = a.direct_ok && a.direct_emit && exclusive && a.slowflag[lo] == 0;
    for (int i = threadIdx.x; i < kPartCap * cs / 16; i += blockDim.x) ((uint4*)tab)[i] = make_uint4(0, 0, 0, 0);
    if (threadIdx.x == 0) overflowed = 0;
    __syncthreads();
    for (int64_t base = s; base < seg_end; base += kAggILP * blockDim.x) {
      uint64_t key[kAggILP];
      int32_t v[kAggILP][NV > 0 ? NV : 1];
      bool valid[kAggILP];
#pragma unroll
      for (int k = 0; k < kAggILP; ++k) {   // loads of kAggILP records first
        const int64_t j = base + k * blockDim.x + threadIdx.x;
        valid[k] = j < seg_end;
        key[k] = 0;
#pragma unroll
        for (int i = 0; i < NV; ++i) v[k][i] = 0;
        if (valid[k]) load_rec<NV>(a.recs + (size_t)j * a.rec_bytes, key[k], v[k]);
      }
#pragma unroll
      for (int k = 0; k < kAggILP; ++k) {
        const uint64_t k0 = __shfl_sync(0xffffffffu, key[k], 0);
        if (__all_sync(0xffffffffu, valid[k] && key[k] == k0)) {    // heavy hitter: one update per warp
          const int ts = __shfl_sync(0xffffffffu, lane == 0 ? part_find(tab, k0, direct, a.pbits) : -1, 0);
          if (ts >= 0) {
            part_add_warp<NV, FIX>(p, tab, ts, v[k], lane);
            continue;
          }
        }
        const int ts = part_find_warp(tab, key[k], valid[k], direct, a.pbits);
        if (!valid[k]) continue;
        if (ts >= 0) {
          part_add<NV, FIX>(p, tab, ts, v[k], a.mm_check != 0);
        } else {
          overflowed = 1;
          if (a.lazy && direct) continue;                      // region not zeroed yet: redone below
          uint8_t* ge = table_find_or_insert(p.table, p.mask, p.stride, key[k], p.status);
          if (ge) update_entry_rec(p, ge, v[k], p.nvals);
        }
      }
    }
    __syncthreads();
    if (a.lazy && direct && overflowed) {
      // shared table overflowed in a partition whose HBM region was left dirty: this CTA is
      // the only one touching the region — clear it and aggregate the whole item there
      uint4* r = (uint4*)(p.table + ((size_t)lo << kPartCapBits) * p.stride);
      const int nq = (int)(((size_t)p.stride << kPartCapBits) / 16);
      for (int i = threadIdx.x; i < nq; i += blockDim.x) r[i] = make_uint4(0, 0, 0, 0);
      __syncthreads();
      for (int64_t j = s + threadIdx.x; j < seg_end; j += blockDim.x) {
        uint64_t key;
        int32_t v[NV > 0 ? NV : 1];
        load_rec<NV>(a.recs + (size_t)j * a.rec_bytes, key, v);
        uint8_t* ge = table_find_or_insert(p.table, p.mask, p.stride, key, p.status);
        if (ge) update_entry_rec(p, ge, v, p.nvals);
      }
    } else if (direct && !overflowed && a.direct_emit) {               // the rows straight from shared memory
      constexpr int PER = kPartCap / kPartThreads;
      uint32_t occ = 0;
#pragma unroll
      for (int k = 0; k < PER; ++k) {
        const int slot = threadIdx.x + k * kPartThreads;
        if (*pkey(tab, slot) != 0 && *pf32(tab, slot, 8) != 0) occ |= 1u << k;
      }
      // occupied slots listed in shared memory, then emitted by consecutive threads into
      // consecutive output rows (coalesced stores)
      const int64_t g0 = part_emit_claim(__popc(occ), a.out_ctr, wsum, &base_s);
      const uint32_t off = (uint32_t)(g0 - (int64_t)base_s);
      uint32_t at = off;
#pragma unroll
      for (int k = 0; k < PER; ++k)
        if ((occ >> k) & 1u) slot_list[at++] = (uint16_t)(threadIdx.x + k * kPartThreads);
      uint32_t tot = 0;
      for (int w = 0; w < kPartThreads / 32; ++w) tot += wsum[w];
      __syncthreads();
      for (uint32_t i = threadIdx.x; i < tot; i += kPartThreads)
        part_emit_row(p, a, ea, tab, slot_list[i], (int64_t)base_s + i);
    } else if (exclusive) {
      for (int i = threadIdx.x; i < kPartCap; i += blockDim.x) part_flush_slot_excl(p, tab, i);
    } else {
      for (int i = threadIdx.x; i < kPartCap; i += blockDim.x) part_flush_slot(p, tab, i);
    }
    if (a.direct_emit && !(direct && !overflowed) && threadIdx.x == 0) a.dirty[lo] = 1;   // rows in the HBM range
    __syncthreads();
  }
}

// Emission of the partitions whose groups live in the HBM table (split / overflowed /
// exact-path partitions): one CTA per partition scans its kPartCap-slot range.
__global__ void __launch_bounds__(kPartThreads) k_part_emit_dirty(const __grid_constant__ Plan p, PartArgs a,
                                                                  const __grid_constant__ EmitArgs ea) {
  __shared__ uint32_t wsum[kPartThreads / 32];
  __shared__ unsigned long long base_s;
  const int64_t q = blockIdx.x;
  if (!a.dirty[q] && !a.slowflag[q]) return;                  // CTA-uniform
  constexpr int PER = kPartCap / kPartThreads;
  const uint8_t* region = p.table + ((size_t)q << kPartCapBits) * p.stride;
  uint32_t occ = 0;
#pragma unroll
  for (int k = 0; k < PER; ++k)
    if (*(const uint64_t*)(region + (size_t)(threadIdx.x + k * kPartThreads) * p.stride) != 0) occ |= 1u << k;
  int64_t g = part_emit_claim(__popc(occ), a.out_ctr, wsum, &base_s);
#pragma unroll
  for (int k = 0; k < PER; ++k)
    if ((occ >> k) & 1u) {
      const uint8_t* e = region + (size_t)(threadIdx.x + k * kPartThreads) * p.stride;
      part_emit_row(ea, p.stride, e, ~*(const uint64_t*)e, g++);
    }
}

// The side entry (key ~0), then the row count and the capacity check.
__global__ void k_part_emit_finish(const __grid_constant__ Plan p, PartArgs a, const __grid_constant__ EmitArgs ea,
                                   int64_t out_capacity) {
  const uint8_t* side = p.table + (p.mask + 1) * (uint64_t)p.stride;
  if (*(const uint64_t*)side) part_emit_row(ea, p.stride, side, ~0ULL, (int64_t)atomicAdd(a.out_ctr, 1ULL));
  const int64_t G = (int64_t)*a.out_ctr;
  *a.count_out = G;
  if (G > out_capacity) set_status(p.status, OCL_ERR_CAPACITY);
}

// ------------------------------------------------------------------ host
using PShK64 = StaticShape<0, false, 8, 0, 1, false, vop(0, VF_SUM | VF_MIN | VF_MAX, 0)>;
using PShP32K64 = StaticShape<4, false, 8, 0, 1, false, vop(0, VF_SUM | VF_MIN | VF_MAX, 0)>;

static int part_rec_bytes(int nv) { return nv <= 2 ? 16 : 32; }

// Pass 1b: 5 = two levels above 2^kPartLevelBits partitions, level 1 into per-block ranges
// (k_part_scatter_l1), level 2 by tiles with direct-indexed maps (default; one tiled level
// below); 0 = one-level scatter with per-row claims, three-stage pipeline (16-byte
// records, else as 4); 4 = one-level, next rows prefetched; 2 / 3 = one-level without the
// prefetch at two CTAs per SM, 4 / 8 rows per thread; 1 = tiled scatter, two levels above
// 2^kPartLevelBits partitions (OCL_PSCAT=1; the round-1/2 design, kept for A/B).
static int part_scatter_mode() {
  const char* e = getenv("OCL_PSCAT");
  return e ? atoi(e) : 5;
}
static size_t align_up(size_t x, size_t a) { return (x + a - 1) / a * a; }

// Partition count: ~1024 expected keys per partition (shared-table load 1/2) while a partition's
// records fit one pass-2 item, so partitions are emitted straight from shared memory (direct
// emission needs the HBM table to hold exactly kPartCap slots per partition).  When items are
// split anyway (many rows per key) and one scatter level suffices, fewer keys per table shorten
// the probe sequences: 256 keys, or 512 if 256 would add the second level.  Measured on C5
// (2^28 rows): 2^12 / 2^14 / 2^16 groups 6.12 / 6.10 / 6.20 -> 4.93 / 5.07 / 5.61 ms.
int part_bits_for(int64_t expected_groups, int64_t n) {
  // at most 2^14 partitions (64 KB count-pass histogram; 2^15 measured slower: C3 2.34 -> 5.82 ms,
  // C5 2^24 groups 8.90 -> 12.4 ms with 512 keys per partition)
  constexpr int maxb = 14;
  auto bits = [&](int64_t per) {
    int b = 0;
    while (b < maxb && (per << b) < expected_groups) ++b;
    return b;
  };
  if (const char* e = getenv("OCL_PART_KEYS")) return bits(std::max(64, std::min(kPartCap / 2, atoi(e))));
  const int b1024 = bits(kPartCap / 2);
  // one-level plans only: with two levels, more partitions cost more than the shorter probes
  // gain (C5 sweep, 2^20-2^22 groups: up to 1.67x slower at 1 % selectivity, where n overstates
  // the records)
  if ((n >> b1024) <= kPartItem || b1024 > kPartLevelBits) return b1024;
  const int b256 = bits(256), b512 = bits(512);
  if (b256 <= kPartLevelBits) return b256;
  return b512 <= kPartLevelBits ? b512 : b1024;
}

static int part_nblk(int sms, int64_t n) {
  // 4 row blocks per SM (the workspace sizes allow no more).  3 / 2 per SM, which would keep the
  // 64 KB-histogram count pass of C3 in one wave, measured slower: C3 2.34 -> 2.51 / 2.50 ms,
  // C5 2^24 groups 8.89 -> 9.77 / 9.77 ms
  int64_t nb = (int64_t)sms * 4;
  const int64_t need = (n + 4095) / 4096;
  return (int)std::max<int64_t>(1, std::min(nb, need));
}

bool part_eligible(const Plan& p) {
  if (p.nkeys < 1 || p.nvals > 6 || p.direct) return false;
  for (int v = 0; v < p.nvals; ++v)
    if (p.vals[v].is_f64 || p.vals[v].expr != OCL_EXPR_COL) return false;
  return true;
}

size_t part_ws_bytes(const Plan& p, int pbits, int sms) {
  const int64_t L = 1LL << pbits;
  const int64_t nchunks = (L + kScanChunk - 1) / kScanChunk;
  const bool two = pbits > kPartLevelBits;
  const size_t n1 = ((size_t)1 << kPartLevelBits) * (size_t)sms * 4;   // level-1 counts per row block (nblk <= 4 sms)
  const size_t sparse = p.npreds > 0 ? align_up((size_t)p.n * 4, 256) + align_up((size_t)sms * 16, 256) + 256 : 0;
  return align_up((size_t)L * 4, 256) * 7 + align_up((size_t)L * 128, 256) + align_up((size_t)nchunks * 4, 256) * 2 + 768 +
         align_up(n1 * 4, 256) + align_up((n1 / kScanChunk + 1) * 4, 256) + sparse +
         align_up((size_t)p.n * part_rec_bytes(p.nvals), 256) * (two ? 2 : 1) + (two ? align_up(4u << kPartLevelBits, 256) : 0);
}

template <class Sh, int NV>
static cudaError_t part_run(const Plan& p, PartArgs a, int sms, cudaStream_t s, const EmitArgs& ea,
                            int64_t out_capacity) {
  const size_t hsm = (size_t)4 << a.pbits;
  auto kc = k_part_count<Sh, NV, false>;
  auto kcs = k_part_count<Sh, NV, true>;
  auto ks = k_part_scatter<Sh, NV>;
  const bool fix = NV == 1 && p.nvals == 1 && p.vals[0].co_lo == 12 && p.vals[0].co_hi == 16 &&
                   p.vals[0].co_min == 20 && p.vals[0].co_max == 24;
  auto ka = fix ? k_part_agg<NV, NV == 1> : k_part_agg<NV, false>;
  cudaError_t e;
  if ((e = cudaFuncSetAttribute(kc, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)hsm))) return e;
  if ((e = cudaFuncSetAttribute(kcs, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)hsm))) return e;
  const size_t tsm = (size_t)kPartCap * p.cta_stride;
  if ((e = cudaFuncSetAttribute(ka, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)tsm))) return e;
  const int64_t L = 1LL << a.pbits;
  const int64_t nchunks = (L + kScanChunk - 1) / kScanChunk;
  if ((e = cudaMemsetAsync(a.counts, 0, (size_t)L * 4, s))) return e;
  if ((e = cudaMemsetAsync(a.slowflag, 0, (size_t)L * 4, s))) return e;
  if (a.direct_emit) {
    if ((e = cudaMemsetAsync(a.dirty, 0, (size_t)L * 4, s))) return e;
    if ((e = cudaMemsetAsync(a.out_ctr, 0, 8, s))) return e;
  }
  a.b1 = std::min(a.pbits, kPartLevelBits);
  if (part_scatter_mode() != 5) a.cnt1 = nullptr;
  if (!a.cnt1 || (getenv("OCL_PART_SPARSE") && atoi(getenv("OCL_PART_SPARSE")) == 0)) a.sparse_dev = nullptr;
  if (a.sparse_dev) {
    count_launch();
    k_part_sample<Sh><<<1, 1024, 0, s>>>(p, a.sparse_dev);
  }
  count_launch(4);
  kc<<<a.nblk, kPartThreads, hsm, s>>>(p, a);
  if (a.sparse_dev) {
    count_launch();
    kcs<<<a.nblk, kPartThreads, hsm, s>>>(p, a);
  }
  k_scan_chunks<<<(int)nchunks, kScanThreads, 0, s>>>(a.counts, a.offs, a.sums, L);
  k_scan_sums<<<1, kScanThreads, 0, s>>>(a.sums, nchunks, a.m_dev);
  k_scan_add<<<(int)((L + 255) / 256), 256, 0, s>>>(a.offs, a.cur, a.sums, L);
  if (a.lazy) {
    count_launch();
    k_part_zero_regions<<<(int)L, 256, 0, s>>>(p, a);
  }
  const int b1 = a.b1, b2 = a.pbits - b1;
  const size_t msm = sizeof(TileMap);
  auto ks2 = k_part_scatter2<NV>;
  const bool l1_512 = getenv("OCL_L1T") && atoi(getenv("OCL_L1T")) == 512;   // A/B: 512-thread level-1 blocks
  auto kl1 = l1_512 ? k_part_scatter_l1<Sh, NV, 512, false> : k_part_scatter_l1<Sh, NV, 256, false>;
  auto kl1s = k_part_scatter_l1<Sh, NV, 256, true>;
  const int l1t = l1_512 ? 512 : 256;
  const size_t l1sm = l1_512 ? sizeof(L1Map<512>) : sizeof(L1Map<256>);
  if ((e = cudaFuncSetAttribute(ks, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)msm))) return e;
  if ((e = cudaFuncSetAttribute(ks2, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)msm))) return e;
  if ((e = cudaFuncSetAttribute(kl1, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)l1sm))) return e;
  if ((e = cudaFuncSetAttribute(kl1s, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sizeof(L1Map<256>)))) return e;
  const int smode = part_scatter_mode();
  if (a.cnt1) {                           // two levels, level 1 into per-block ranges
    const int64_t n1 = ((int64_t)1 << b1) * a.nblk, nc1 = (n1 + kScanChunk - 1) / kScanChunk;
    count_launch(4);
    k_scan_chunks<<<(int)nc1, kScanThreads, 0, s>>>(a.cnt1, a.cnt1, a.sums1, n1);
    k_scan_sums<<<1, kScanThreads, 0, s>>>(a.sums1, nc1, a.nitems_dev);     // (total unused; rewritten below)
    k_scan_add<<<(int)((n1 + 255) / 256), 256, 0, s>>>(a.cnt1, a.cnt1, a.sums1, n1);
    uint8_t* l1out = b2 == 0 ? a.recs : a.tmp;   // one level: the per-block ranges are the final partitions
    kl1<<<a.nblk, l1t, l1sm, s>>>(p, a, l1out);
    if (a.sparse_dev) {
      count_launch();
      kl1s<<<a.nblk, 256, sizeof(L1Map<256>), s>>>(p, a, l1out);
    }
    if (b2 != 0) {
      count_launch();
      ks2<<<a.nblk, kPartThreads, msm, s>>>(a);
    }
  } else if (smode != 1 && smode != 5) {
    count_launch(2);
    k_part_cur_pad<<<(int)((L + 255) / 256), 256, 0, s>>>(a.offs, a.curp, a.curp_shift, L);
    if (smode == 0 && NV <= 2) k_part_scatter_pipe<Sh, NV <= 2 ? NV : 2><<<a.nblk, kPartThreads, 0, s>>>(p, a);
    else if (smode == 0 || smode == 4) k_part_scatter_direct<Sh, NV, true, 1><<<a.nblk, kPartThreads, 0, s>>>(p, a);
    else if (smode == 2) k_part_scatter_direct<Sh, NV, false, 1><<<a.nblk, kPartThreads, 0, s>>>(p, a);
    else k_part_scatter_direct<Sh, NV, false, 2><<<a.nblk, kPartThreads, 0, s>>>(p, a);
  } else if (b2 == 0) {
    ks<<<a.nblk, kPartThreads, msm, s>>>(p, a, a.pbits, a.cur, a.recs);
  } else {
    count_launch(3);
    k_part_cur1<<<((1 << b1) + 255) / 256, 256, 0, s>>>(a.offs, a.cur1, b1, b2);
    ks<<<a.nblk, kPartThreads, msm, s>>>(p, a, b1, a.cur1, a.tmp);
    ks2<<<a.nblk, kPartThreads, msm, s>>>(a);
  }
  count_launch(4);
  k_part_items<<<(int)((L + 255) / 256), 256, 0, s>>>(a);
  k_scan_chunks<<<(int)nchunks, kScanThreads, 0, s>>>(a.icnt, a.ioff, a.isums, L);
  k_scan_sums<<<1, kScanThreads, 0, s>>>(a.isums, nchunks, a.nitems_dev);
  k_scan_add<<<(int)((L + 255) / 256), 256, 0, s>>>(a.ioff, a.icnt, a.isums, L);   // icnt := ioff (unused after)
  int nb = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&nb, ka, kPartThreads, tsm) != cudaSuccess || nb < 1) nb = 1;
  const int64_t items = (p.n + kPartItem - 1) / kPartItem + L;
  const int64_t grid = std::max<int64_t>(1, std::min<int64_t>((int64_t)sms * nb, items));
  count_launch();
  ka<<<(int)grid, kPartThreads, tsm, s>>>(p, a, ea);
  if (a.direct_emit) {
    count_launch(2);
    k_part_emit_dirty<<<(int)L, kPartThreads, 0, s>>>(p, a, ea);
    k_part_emit_finish<<<1, 1, 0, s>>>(p, a, ea, out_capacity);
  }
  return cudaGetLastError();
}

// Run the partitioned tier for plan p (p.table NOT zeroed by the caller: done here, fully or
// lazily; p.n > 0).  *kind reports
// the shape (30 dynamic, 31 key i64, 32 pred i32 + key i64).
cudaError_t launch_partitioned(const Plan& p, int pbits, void* ws, int sms, cudaStream_t s, int* kind,
                               const EmitArgs* ea, int64_t* count_out, int64_t out_capacity, bool* emitted) {
  if (emitted) *emitted = false;
  if (p.n == 0) return cudaSuccess;
  PartArgs a;
  a.pbits = pbits;
  a.nblk = part_nblk(sms, p.n);
  a.rows_per_blk = ((p.n + a.nblk - 1) / a.nblk + 127) / 128 * 128;
  const int64_t L = 1LL << pbits;
  const int64_t nchunks = (L + kScanChunk - 1) / kScanChunk;
  uint8_t* w = (uint8_t*)ws;
  a.counts = (uint32_t*)w;
  w += align_up((size_t)L * 4, 256);
  a.offs = (uint32_t*)w;
  w += align_up((size_t)L * 4, 256);
  a.cur = (uint32_t*)w;
  w += align_up((size_t)L * 4, 256);
  a.sums = (uint32_t*)w;
  w += align_up((size_t)nchunks * 4, 256);
  a.icnt = (uint32_t*)w;
  w += align_up((size_t)L * 4, 256);
  a.ioff = (uint32_t*)w;
  w += align_up((size_t)L * 4, 256);
  a.isums = (uint32_t*)w;
  w += align_up((size_t)nchunks * 4, 256);
  a.nitems_dev = (int64_t*)w;
  w += 256;
  a.slowflag = (uint32_t*)w;
  w += align_up((size_t)L * 4, 256);
  a.direct_ok = ((p.mask + 1) >> pbits) == (uint64_t)kPartCap ? 1 : 0;
  a.m_dev = (int64_t*)w;
  w += 256;
  a.rec_bytes = part_rec_bytes(p.nvals);
  a.recs = w;
  w += align_up((size_t)p.n * a.rec_bytes, 256);
  a.tmp = nullptr;
  a.cur1 = nullptr;
  if (pbits > kPartLevelBits) {
    a.tmp = w;
    w += align_up((size_t)p.n * a.rec_bytes, 256);
    a.cur1 = (uint32_t*)w;
    w += align_up(4u << kPartLevelBits, 256);
  }
  a.dirty = (uint32_t*)w;
  w += align_up((size_t)L * 4, 256);
  a.curp = (uint32_t*)w;
  w += align_up((size_t)L * 128, 256);
  {
    const size_t n1 = ((size_t)1 << kPartLevelBits) * (size_t)sms * 4;
    a.cnt1 = (uint32_t*)w;
    w += align_up(n1 * 4, 256);
    a.sums1 = (uint32_t*)w;
    w += align_up((n1 / kScanChunk + 1) * 4, 256);
  }
  a.sparse_dev = nullptr;
  a.soids = nullptr;
  a.nq = nullptr;
  if (p.npreds > 0) {
    a.soids = (uint32_t*)w;
    w += align_up((size_t)p.n * 4, 256);
    a.nq = (uint32_t*)w;
    w += align_up((size_t)sms * 16, 256);
    a.sparse_dev = (int32_t*)w;
    w += 256;
  }
  a.curp_shift = 0;                                     // packed (padding to a sector or line measured slower)
  if (const char* cp = getenv("OCL_CURPAD")) a.curp_shift = std::min(5, std::max(0, atoi(cp)));
  a.out_ctr = (unsigned long long*)w;
  a.count_out = count_out;
  a.direct_emit = (ea && count_out && a.direct_ok && p.stride <= 256) ? 1 : 0;
  a.lazy = 0;
  a.mm_check = 0;                                       // C3 uniform: 3.09 (on) -> 3.02 ms (off)
  if (const char* mc = getenv("OCL_MM_CHECK")) a.mm_check = atoi(mc) != 0;
  EmitArgs none;
  memset(&none, 0, sizeof(none));
  const EmitArgs& e = ea ? *ea : none;
  a.npo = 0;
  if (a.direct_emit && e.kind == EMIT_FINAL) {            // outputs resolved once, not per row
    for (int i = 0; i < e.fin.naggs; ++i) {
      const OutAgg& o = e.fin.aggs[i];
      auto& q = a.po[a.npo];
      q.out = o.out;
      q.f0 = q.f1 = 0;
      q.kind = -1;
      if (o.op == OCL_AGG_COUNT) q.kind = 0;
      for (int v = 0; v < p.nvals && q.kind < 0; ++v) {
        const DevValue& d = p.vals[v];
        if ((o.op == OCL_AGG_SUM || o.op == OCL_AGG_AVG) && o.off == d.off_sum) {
          q.kind = o.op == OCL_AGG_SUM ? 1 : 2;
          q.f0 = d.co_lo;
          q.f1 = d.co_hi;
        } else if (o.op == OCL_AGG_MIN && o.off == d.off_min) {
          q.kind = 3;
          q.f0 = d.co_min;
        } else if (o.op == OCL_AGG_MAX && o.off == d.off_max) {
          q.kind = 4;
          q.f0 = d.co_max;
        }
      }
      if (q.kind < 0) a.direct_emit = 0;                    // unexpected aggregate: the table path
      ++a.npo;
    }
  }
  if (emitted) *emitted = a.direct_emit != 0;
  // The HBM table (cap + 1 entries; the caller leaves it unzeroed): with direct emission only
  // the regions that receive entries are cleared on the device (k_part_zero_regions, the
  // overflow branch of k_part_agg) and the side entry here; otherwise all of it.
  a.lazy = a.direct_emit && getenv("OCL_PART_EAGER") == nullptr ? 1 : 0;
  {
    const size_t tb = (size_t)(p.mask + 2) * p.stride;
    cudaError_t ze = a.lazy ? cudaMemsetAsync(p.table + (size_t)(p.mask + 1) * p.stride, 0, p.stride, s)
                            : cudaMemsetAsync(p.table, 0, tb, s);
    if (ze) return ze;
  }
  if (p.vec_ok && p.nkeys == 1 && p.npreds == 0 && values_match<PShK64>(p) && p.keys[0].col.width == 8) {
    *kind = 31;
    return part_run<PShK64, 1>(p, a, sms, s, e, out_capacity);
  }
  if (p.vec_ok && p.nkeys == 1 && p.npreds == 1 && p.preds[0].col.width == 4 && !p.preds[0].is_f64 &&
      values_match<PShP32K64>(p) && p.keys[0].col.width == 8) {
    *kind = 32;
    return part_run<PShP32K64, 1>(p, a, sms, s, e, out_capacity);
  }
  *kind = 30;
  if (p.nvals <= 1) return part_run<DynShape, 1>(p, a, sms, s, e, out_capacity);
  if (p.nvals <= 2) return part_run<DynShape, 2>(p, a, sms, s, e, out_capacity);
  if (p.nvals <= 4) return part_run<DynShape, 4>(p, a, sms, s, e, out_capacity);
  return part_run<DynShape, 6>(p, a, sms, s, e, out_capacity);
}

}  // namespace ocl
