// fused.cu — K9: fused select -> hash group -> aggregate, one pass over the columns.
//
// Paper steps fused here: selection (§4.1.1), hash group-by
// with dense group ids (L551-561 §4.1.6; hashing L511-533 §4.1.4), multi-column
// grouping on combined ids (L559-561), hierarchical grouped aggregation with
// per-work-group tables and several accumulators per group for few groups
// (L562-600 §4.1.7).  Nothing is materialised: no bitmap (unless requested for
// tests), no oid list, no gid column.
//
// B200 design:
//  * persistent grid (#SMs x resident CTAs); a warp owns tiles of 64*U rows; lane
//    l handles rows (2l, 2l+1) of each 64-row unit, so every column is read with one
//    vector load per lane per unit (u8: 2 B, i32: 8 B, i64/f64: 16 B) and every
//    warp-wide load is a contiguous, fully-used run (P:L619-633 GPU pattern).
//  * REGISTER tier (few groups): each thread keeps L private accumulator slots in
//    registers — the limit of the paper's "multiple accumulators per group" idea:
//    one accumulator set per thread, no atomics in the row loop.  A block-wide
//    slot directory in shared memory gives every thread the same key -> slot map.
//    Integer SUMs use 96-bit (lo64 + hi32) predicated add-with-carry chains: exact
//    for any per-thread row count < 2^31 (the int128 state is formed at flush).
//  * GLOBAL tier (many groups): find-or-insert in the HBM open-addressing table
//    and update the entry with atomics (native f64 add, int128 as two u64 atomics).
//  * Rows a tier cannot place (more than L keys in a block, int32-overflowing
//    factors, the key ~0) take the exact int128 global path, so every tier is
//    correct for every input; the tier only decides speed.
#include "launch.cuh"
#include "rowops.cuh"

namespace ocl {

constexpr int kFusedThreads = 256;

__device__ __forceinline__ void add96(bool pr, uint32_t& a0, uint32_t& a1, uint32_t& a2, int64_t v) {
  uint32_t v0 = (uint32_t)(uint64_t)v, v1 = (uint32_t)((uint64_t)v >> 32), v2 = (uint32_t)(v >> 63);
  asm("{\n\t.reg .pred p;\n\t"
      "setp.ne.u32 p, %3, 0;\n\t"
      "@p add.cc.u32 %0, %0, %4;\n\t"
      "@p addc.cc.u32 %1, %1, %5;\n\t"
      "@p addc.u32 %2, %2, %6;\n\t}"
      : "+r"(a0), "+r"(a1), "+r"(a2)
      : "r"((uint32_t)pr), "r"(v0), "r"(v1), "r"(v2));
}

// Per-row inputs after predicate / key / value evaluation.
template <int NV, bool F64>
struct RowIn {
  bool q;
  bool fast;
  uint64_t key;
  int64_t vi[F64 ? 1 : NV];
  double vd[F64 ? NV : 1];
};

// Evaluate values of one row from raw operands (vector path: loaded as pairs).
template <int NV, bool F64>
__device__ __forceinline__ void eval_values_pair(const Plan& p, int64_t r, RowIn<NV, F64>& x0, RowIn<NV, F64>& x1) {
#pragma unroll
  for (int v = 0; v < NV; ++v) {
    if (v >= p.nvals) break;
    const DevValue& d = p.vals[v];
    if constexpr (!F64) {
      if (d.is_f64) {   // mixed int/fp64 plan: fp64 values take the exact slow path
        x0.fast = x1.fast = false;
        continue;
      }
    }
    uint64_t a0, a1, b0 = 0, b1 = 0, c0 = 0, c1 = 0;
    load_pair(d.a, r, a0, a1);
    if (d.expr >= OCL_EXPR_MUL_1MINUS) load_pair(d.b, r, b0, b1);
    if (d.expr >= OCL_EXPR_MUL_1MINUS_1PLUS) load_pair(d.c, r, c0, c1);
    if constexpr (F64) {
      x0.vd[v] = value_f64(d, a0, b0, c0);
      x1.vd[v] = value_f64(d, a1, b1, c1);
    } else {
      x0.vi[v] = value_i64_fast(d, a0, b0, c0, x0.fast);
      x1.vi[v] = value_i64_fast(d, a1, b1, c1, x1.fast);
    }
  }
}

template <int NV, bool F64>
__device__ __forceinline__ void eval_row_scalar(const Plan& p, int64_t r, RowIn<NV, F64>& x) {
  x.fast = true;
  x.q = r < p.n && row_pred_scalar(p, r);
  x.key = 0;
  if (!x.q) return;
  x.key = row_key_scalar(p, r);
#pragma unroll
  for (int v = 0; v < NV; ++v) {
    if (v >= p.nvals) break;
    const DevValue& d = p.vals[v];
    if constexpr (!F64) {
      if (d.is_f64) {
        x.fast = false;
        continue;
      }
    }
    uint64_t a = load_one(d.a, r);
    uint64_t b = d.expr >= OCL_EXPR_MUL_1MINUS ? load_one(d.b, r) : 0;
    uint64_t c = d.expr >= OCL_EXPR_MUL_1MINUS_1PLUS ? load_one(d.c, r) : 0;
    if constexpr (F64) x.vd[v] = value_f64(d, a, b, c);
    else x.vi[v] = value_i64_fast(d, a, b, c, x.fast);
  }
}

template <int NV, bool F64>
__device__ __forceinline__ void eval_pair_vec(const Plan& p, int64_t r, RowIn<NV, F64>& x0, RowIn<NV, F64>& x1) {
  x0.q = true;
  x1.q = true;
#pragma unroll
  for (int i = 0; i < kMaxPreds; ++i) {
    if (i >= p.npreds) break;
    uint64_t u0, u1;
    load_pair(p.preds[i].col, r, u0, u1);
    x0.q = x0.q && eval_pred(p.preds[i], u0);
    x1.q = x1.q && eval_pred(p.preds[i], u1);
  }
  x0.key = 0;
  x1.key = 0;
#pragma unroll
  for (int i = 0; i < kMaxKeys; ++i) {
    if (i >= p.nkeys) break;
    uint64_t u0, u1;
    load_pair(p.keys[i].col, r, u0, u1);
    x0.key |= (u0 & p.keys[i].mask) << p.keys[i].shift;
    x1.key |= (u1 & p.keys[i].mask) << p.keys[i].shift;
  }
  x0.fast = true;
  x1.fast = true;
  eval_values_pair<NV, F64>(p, r, x0, x1);
}

// ------------------------------------------------------------------ register (private accumulator) tier
// Few groups: each thread owns one accumulator record per group slot in shared
// memory, laid out [slot][field][thread] (field offsets from the host planner,
// Plan::priv_rec bytes per thread per slot): count u32; per value: SUM as 96-bit
// (u64 lo + u32 hi) or double; MIN / MAX as order-preserving u64 encodings (zero
// = identity).  A row costs one slot-indexed read-modify-write per accumulator:
// no atomics in the row loop — the limit of the paper's "multiple accumulators
// per group" in local memory.  A block-wide slot directory in shared
// memory gives every thread the same key -> slot map.
constexpr int kRegSlots = 4;

template <int NV, bool F64>
__device__ __forceinline__ void privg_add(const Plan& p, uint8_t* sm, int slot, int tid, const RowIn<NV, F64>& x) {
  constexpr int T = kFusedThreads;
  uint8_t* base = sm + (size_t)slot * p.priv_rec * T;
  ((uint32_t*)base)[tid] += 1u;
#pragma unroll
  for (int v = 0; v < NV; ++v) {
    if (v >= p.nvals) break;
    const DevValue& d = p.vals[v];
    if constexpr (F64) {
      const double val = x.vd[v];
      if (d.po_sum >= 0) ((double*)(base + d.po_sum * T))[tid] += val;
      if (d.po_min >= 0) {
        uint64_t* m = (uint64_t*)(base + d.po_min * T) + tid;
        *m = max(*m, enc_min_f(val));
      }
      if (d.po_max >= 0) {
        uint64_t* m = (uint64_t*)(base + d.po_max * T) + tid;
        *m = max(*m, enc_max_f(val));
      }
    } else {
      if (d.is_f64) continue;                       // mixed plan: fp64 values went to the slow path
      const int64_t val = x.vi[v];
      if (d.po_sum >= 0) {
        uint64_t* lo = (uint64_t*)(base + d.po_sum * T) + tid;
        uint32_t* hi = (uint32_t*)(base + d.po_hi * T) + tid;
        uint64_t l = *lo;
        uint32_t h = *hi;
        uint32_t l0 = (uint32_t)l, l1 = (uint32_t)(l >> 32);
        asm("add.cc.u32 %0, %0, %3;\n\taddc.cc.u32 %1, %1, %4;\n\taddc.u32 %2, %2, %5;"
            : "+r"(l0), "+r"(l1), "+r"(h)
            : "r"((uint32_t)(uint64_t)val), "r"((uint32_t)((uint64_t)val >> 32)), "r"((uint32_t)(val >> 63)));
        *lo = (uint64_t)l0 | ((uint64_t)l1 << 32);
        *hi = h;
      }
      if (d.po_min >= 0) {
        uint64_t* m = (uint64_t*)(base + d.po_min * T) + tid;
        *m = max(*m, enc_min_i(val));
      }
      if (d.po_max >= 0) {
        uint64_t* m = (uint64_t*)(base + d.po_max * T) + tid;
        *m = max(*m, enc_max_i(val));
      }
    }
  }
}

// Per-CTA shared-memory hash table (mid G: more distinct keys than private slots;
// the paper's per-work-group local-memory aggregation tables).
// sm_100 has no native 64-bit shared-memory atomic add/max (they lower to CAS
// loops), so the table uses 32-bit fields and native 32-bit atomics only:
//   [~key u64][count u32] per value: [sum of low 16 bits u32][sum of high 16 bits s32]
//   [min u32][max u32] (order-preserving encodings, 0 = identity).
// Values are int32 on this path (fast-path COL values), so each field absorbs 2^16
// updates exactly; the CTA flushes the table into the HBM table every 2^16 rows.
// Linear probing with 64-bit shared atomicCAS on the key, at most kSmemProbes probes.
constexpr int kSmemProbes = 16;
constexpr int kCtaFlushRounds = 64;   // rounds of (warps x tile) rows = 64 x 8 x 128 = 65,536 rows

__device__ __forceinline__ uint8_t* smem_find_or_insert(uint8_t* tab, uint32_t cap, int32_t stride, uint64_t key) {
  const uint64_t sk = ~key;
  uint32_t h = (uint32_t)fmix64(key) & (cap - 1);
  for (int probe = 0; probe < kSmemProbes; ++probe) {
    uint64_t* kp = (uint64_t*)(tab + (size_t)h * stride);
    uint64_t cur = *(volatile uint64_t*)kp;
    if (cur == sk) return (uint8_t*)kp;
    if (cur == 0) {
      uint64_t prev = atomicCAS((unsigned long long*)kp, 0ULL, (unsigned long long)sk);
      if (prev == 0 || prev == sk) return (uint8_t*)kp;
    }
    h = (h + 1) & (cap - 1);
  }
  return nullptr;
}

__device__ __forceinline__ uint32_t enc32_max(int32_t v) { return (uint32_t)v ^ 0x80000000u; }
__device__ __forceinline__ uint32_t enc32_min(int32_t v) { return ~enc32_max(v); }

template <int NV, bool F64>
__device__ __forceinline__ void cta_add(const Plan& p, uint8_t* e, const RowIn<NV, F64>& x) {
  atomicAdd((unsigned int*)(e + 8), 1u);
  if constexpr (!F64) {
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      if (v >= p.nvals) break;
      const DevValue& d = p.vals[v];
      const int32_t w = (int32_t)x.vi[v];
      if (d.co_lo >= 0) {
        atomicAdd((unsigned int*)(e + d.co_lo), (unsigned int)w & 0xFFFFu);
        atomicAdd((int*)(e + d.co_hi), w >> 16);
      }
      if (d.co_min >= 0) atomicMax((unsigned int*)(e + d.co_min), enc32_min(w));
      if (d.co_max >= 0) atomicMax((unsigned int*)(e + d.co_max), enc32_max(w));
    }
  }
}

// Fold one CTA-table entry into the HBM table and reset its accumulators (key kept).
__device__ __forceinline__ void cta_flush_entry(const Plan& p, uint8_t* ce) {
  const uint64_t sk = *(const uint64_t*)ce;
  const uint32_t cnt = *(const uint32_t*)(ce + 8);
  if (sk == 0 || cnt == 0) return;
  uint8_t* e = table_find_or_insert(p.table, p.mask, p.stride, ~sk, p.status);
  if (e) {
    atomicAdd((unsigned long long*)(e + 8), (unsigned long long)cnt);
    for (int v = 0; v < p.nvals; ++v) {
      const DevValue& d = p.vals[v];
      if (d.co_lo >= 0) {
        const int64_t sum = (int64_t)(*(const int32_t*)(ce + d.co_hi)) * 65536 + (int64_t)(*(const uint32_t*)(ce + d.co_lo));
        atomic_add_i128((uint64_t*)(e + d.off_sum), (uint64_t)sum, (uint64_t)(sum >> 63));
      }
      if (d.co_min >= 0) {
        const int32_t mn = (int32_t)(~*(const uint32_t*)(ce + d.co_min) ^ 0x80000000u);
        atomicMax((unsigned long long*)(e + d.off_min), (unsigned long long)enc_min_i(mn));
      }
      if (d.co_max >= 0) {
        const int32_t mx = (int32_t)(*(const uint32_t*)(ce + d.co_max) ^ 0x80000000u);
        atomicMax((unsigned long long*)(e + d.off_max), (unsigned long long)enc_max_i(mx));
      }
    }
  }
  for (int w = 8; w < p.cta_stride; w += 4) *(uint32_t*)(ce + w) = 0;
}

// Merge a whole entry (shared-memory table or CTA block entry) into the HBM table.
__device__ __forceinline__ void entry_merge_global(const Plan& p, uint64_t key, const uint8_t* src) {
  uint8_t* e = table_find_or_insert(p.table, p.mask, p.stride, key, p.status);
  if (!e) return;
  atomicAdd((unsigned long long*)(e + 8), (unsigned long long)*(const uint64_t*)(src + 8));
  for (int v = 0; v < p.nvals; ++v) {
    const DevValue& d = p.vals[v];
    if (d.off_sum >= 0) {
      if (d.is_f64) atomicAdd((double*)(e + d.off_sum), *(const double*)(src + d.off_sum));
      else atomic_add_i128((uint64_t*)(e + d.off_sum), *(const uint64_t*)(src + d.off_sum),
                           *(const uint64_t*)(src + d.off_sum + 8));
    }
    if (d.off_min >= 0) atomicMax((unsigned long long*)(e + d.off_min), *(const unsigned long long*)(src + d.off_min));
    if (d.off_max >= 0) atomicMax((unsigned long long*)(e + d.off_max), *(const unsigned long long*)(src + d.off_max));
  }
}

// Per-warp staging of rows that miss the private slots: the warp groups them by key
// (__match_any_sync) and one leader per distinct key applies the group's combined
// contribution to the HBM table — hot keys of skewed (Zipf) inputs and runs of
// clustered keys cost one atomic update per warp instead of one per row.
template <int NV, bool F64>
struct MissStage {
  int64_t vi[F64 ? 1 : NV][32];
  double vd[F64 ? NV : 1][32];
};

template <int NV, bool F64>
__device__ __forceinline__ void warp_miss_update(const Plan& p, MissStage<NV, F64>& st, bool miss, const RowIn<NV, F64>& x,
                                                 int lane) {
  const unsigned mmask = __ballot_sync(0xffffffffu, miss);
  if (mmask == 0) return;
  if (miss) {
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      if constexpr (F64) st.vd[v][lane] = x.vd[v];
      else st.vi[v][lane] = x.vi[v];
    }
  }
  __syncwarp();
  if (miss) {
    const unsigned peers = __match_any_sync(mmask, x.key);
    if (lane == __ffs(peers) - 1) {
      uint8_t* e = table_find_or_insert(p.table, p.mask, p.stride, x.key, p.status);
      if (e) {
        atomicAdd((unsigned long long*)(e + 8), (unsigned long long)__popc(peers));
#pragma unroll
        for (int v = 0; v < NV; ++v) {
          if (v >= p.nvals) break;
          const DevValue& d = p.vals[v];
          if constexpr (F64) {
            double sum = 0.0, mn = x.vd[v], mx = x.vd[v];
            for (unsigned b = peers; b; b &= b - 1) {
              const double y = st.vd[v][__ffs(b) - 1];
              sum += y;
              mn = fmin(mn, y);
              mx = fmax(mx, y);
            }
            if (d.off_sum >= 0) atomicAdd((double*)(e + d.off_sum), sum);
            if (d.off_min >= 0) atomicMax((unsigned long long*)(e + d.off_min), (unsigned long long)enc_min_f(mn));
            if (d.off_max >= 0) atomicMax((unsigned long long*)(e + d.off_max), (unsigned long long)enc_max_f(mx));
          } else {
            if (d.is_f64) continue;
            I128 sum{0, 0};
            int64_t mn = x.vi[v], mx = x.vi[v];
            for (unsigned b = peers; b; b &= b - 1) {
              const int64_t y = st.vi[v][__ffs(b) - 1];
              sum = i128_add(sum, i128_from_i64(y));
              mn = min(mn, y);
              mx = max(mx, y);
            }
            if (d.off_sum >= 0) atomic_add_i128((uint64_t*)(e + d.off_sum), sum.lo, sum.hi);
            if (d.off_min >= 0) atomicMax((unsigned long long*)(e + d.off_min), (unsigned long long)enc_min_i(mn));
            if (d.off_max >= 0) atomicMax((unsigned long long*)(e + d.off_max), (unsigned long long)enc_max_i(mx));
          }
        }
      }
    }
  }
  __syncwarp();
}

template <int NV, bool F64>
__device__ __forceinline__ void privg_row(const Plan& p, uint64_t* dir, uint64_t (&rk)[kRegSlots], uint8_t* sm, int tid,
                                          MissStage<NV, F64>& stage, const RowIn<NV, F64>& x, int64_t r) {
  constexpr int L = kRegSlots;
  int slot = -1;
#pragma unroll
  for (int s = L - 1; s >= 0; --s)
    if (x.key == rk[s]) slot = s;
  const bool special = x.key == ~0ULL;
  bool go = x.q && x.fast && slot >= 0 && !special;
  bool miss = false;
  if (x.q && !go) {                       // new key in this CTA, a slow value, or more keys than slots
    slot = (x.fast && !special) ? dir_find_or_insert<L>(dir, x.key) : -1;
    if (slot >= 0) {
#pragma unroll
      for (int s = 0; s < L; ++s) rk[s] = ~*(volatile uint64_t*)&dir[s];
      go = true;
    } else {
      uint8_t* e = nullptr;
      if (p.smem_cap && x.fast && !special)     // mid G: CTA shared-memory table
        e = smem_find_or_insert(sm + (size_t)kRegSlots * p.priv_rec * kFusedThreads, (uint32_t)p.smem_cap,
                                p.cta_stride, x.key);
      if (e) {
        cta_add<NV, F64>(p, e, x);
      } else if (x.fast && !special) {
        miss = true;                            // warp-aggregated HBM update below
      } else {
        e = table_find_or_insert(p.table, p.mask, p.stride, x.key, p.status);
        if (e) update_entry_slow(p, e, r);
      }
    }
  }
  if (go) privg_add<NV, F64>(p, sm, slot, tid, x);
  warp_miss_update<NV, F64>(p, stage, miss, x, tid & 31);
}

template <int NV, bool F64, int U>
__global__ void __launch_bounds__(kFusedThreads) k_sga_reg(const __grid_constant__ Plan p) {
  constexpr int L = kRegSlots;
  constexpr int T = kFusedThreads;
  extern __shared__ __align__(16) uint8_t sm[];
  __shared__ uint64_t dir[L];
  __shared__ __align__(16) uint64_t blk[L * 32];   // block accumulators, entry layout (stride <= 256 B)
  const int tid = threadIdx.x, lane = tid & 31;
  {
    uint4* z = (uint4*)sm;
    const int n16 = (int)(((size_t)L * p.priv_rec * T + (size_t)p.smem_cap * p.cta_stride) / 16);
    for (int i = tid; i < n16; i += T) z[i] = make_uint4(0, 0, 0, 0);
  }
  for (int i = tid; i < L * 32; i += T) blk[i] = 0;
  if (tid < L) dir[tid] = 0;
  __syncthreads();
  uint64_t rk[L];
#pragma unroll
  for (int s = 0; s < L; ++s) rk[s] = ~0ULL;   // ~0 never matches a slot (special key)
  __shared__ MissStage<NV, F64> stages[kFusedThreads / 32];
  MissStage<NV, F64>& stage = stages[tid >> 5];

  constexpr int kTile = 64 * U;
  const int64_t warp = (blockIdx.x * (int64_t)T + tid) >> 5;
  const int64_t nwarps = ((int64_t)gridDim.x * T) >> 5;
  const int64_t ntiles = (p.n + kTile - 1) / kTile;
  // CTA-uniform round count (warp 0 of the CTA has the most tiles) so the whole CTA
  // can meet at the periodic CTA-table flushes
  const int64_t first = (int64_t)blockIdx.x * (T / 32);
  const int64_t rounds = ntiles > first ? (ntiles - first + nwarps - 1) / nwarps : 0;
  uint8_t* cta_tab = sm + (size_t)L * p.priv_rec * T;
  for (int64_t round = 0; round < rounds; ++round) {
    if (p.smem_cap && round > 0 && round % kCtaFlushRounds == 0) {
      __syncthreads();
      for (int i = tid; i < p.smem_cap; i += T) cta_flush_entry(p, cta_tab + (size_t)i * p.cta_stride);
      __syncthreads();
    }
    const int64_t t = warp + round * nwarps;
    if (t >= ntiles) continue;
    const int64_t base = t * kTile;
    const bool vec = p.vec_ok && base + kTile <= p.n;
#pragma unroll
    for (int u = 0; u < U; ++u) {
      const int64_t r = base + 64 * u + 2 * lane;
      RowIn<NV, F64> x0, x1;
      if (vec) {
        eval_pair_vec<NV, F64>(p, r, x0, x1);
      } else {
        eval_row_scalar<NV, F64>(p, r, x0);
        eval_row_scalar<NV, F64>(p, r + 1, x1);
      }
      if (p.bitmap_out) emit_bitmap_unit(p, base + 64 * u, lane, x0.q, x1.q);
      privg_row<NV, F64>(p, dir, rk, sm, tid, stage, x0, r);
      privg_row<NV, F64>(p, dir, rk, sm, tid, stage, x1, r + 1);
    }
  }

  // ---- flush: warp reduce of the private records -> shared block entry -> one global update per slot
  __syncthreads();
  uint8_t* blkb = (uint8_t*)blk;
  for (int s = 0; s < L; ++s) {
    if (dir[s] == 0) continue;                       // uniform: slot never used in this block
    uint8_t* be = blkb + s * 256;
    const uint8_t* rec = sm + (size_t)s * p.priv_rec * T;
    uint32_t c = __reduce_add_sync(0xffffffffu, ((const uint32_t*)rec)[tid]);
    if (lane == 0) atomicAdd((unsigned long long*)(be + 8), (unsigned long long)c);
    for (int v = 0; v < p.nvals; ++v) {
      const DevValue& d = p.vals[v];
      if (d.po_sum >= 0) {
        if (d.is_f64) {
          double sum = ((const double*)(rec + d.po_sum * T))[tid];
          for (int o = 16; o > 0; o >>= 1) sum += __shfl_xor_sync(0xffffffffu, sum, o);
          if (lane == 0) atomicAdd((double*)(be + d.off_sum), sum);
        } else {
          I128 x;
          x.lo = ((const uint64_t*)(rec + d.po_sum * T))[tid];
          x.hi = (uint64_t)(int64_t)(int32_t)((const uint32_t*)(rec + d.po_hi * T))[tid];
          x = warp_sum_i128(x);
          if (lane == 0) atomic_add_i128((uint64_t*)(be + d.off_sum), x.lo, x.hi);
        }
      }
      if (d.po_min >= 0) {
        unsigned long long m = ((const uint64_t*)(rec + d.po_min * T))[tid];
        for (int o = 16; o > 0; o >>= 1) m = max(m, __shfl_xor_sync(0xffffffffu, m, o));
        if (lane == 0 && m) atomicMax((unsigned long long*)(be + d.off_min), m);
      }
      if (d.po_max >= 0) {
        unsigned long long m = ((const uint64_t*)(rec + d.po_max * T))[tid];
        for (int o = 16; o > 0; o >>= 1) m = max(m, __shfl_xor_sync(0xffffffffu, m, o));
        if (lane == 0 && m) atomicMax((unsigned long long*)(be + d.off_max), m);
      }
    }
  }
  __syncthreads();
  // one thread per slot pushes the block entry into the global table
  if (tid < L) {
    const uint64_t sk = dir[tid];
    if (sk != 0) entry_merge_global(p, ~sk, blkb + tid * 256);
  }
  // the CTA's shared-memory table (mid-G): one thread per occupied entry
  if (p.smem_cap)
    for (int i = tid; i < p.smem_cap; i += T) cta_flush_entry(p, cta_tab + (size_t)i * p.cta_stride);
}

// ------------------------------------------------------------------ global tier
template <int NV, bool F64>
__device__ __forceinline__ void glb_row(const Plan& p, const RowIn<NV, F64>& x, int64_t r) {
  if (!x.q) return;
  uint8_t* e = table_find_or_insert(p.table, p.mask, p.stride, x.key, p.status);
  if (!e) return;
  if (!x.fast) {
    update_entry_slow(p, e, r);
    return;
  }
  atomicAdd((unsigned long long*)(e + 8), 1ULL);
#pragma unroll
  for (int v = 0; v < NV; ++v) {
    if (v >= p.nvals) break;
    const DevValue& d = p.vals[v];
    if constexpr (F64) {
      if (d.off_sum >= 0) atomicAdd((double*)(e + d.off_sum), x.vd[v]);
      if (d.off_min >= 0) atomicMax((unsigned long long*)(e + d.off_min), (unsigned long long)enc_min_f(x.vd[v]));
      if (d.off_max >= 0) atomicMax((unsigned long long*)(e + d.off_max), (unsigned long long)enc_max_f(x.vd[v]));
    } else {
      if (d.off_sum >= 0) atomic_add_i128((uint64_t*)(e + d.off_sum), (uint64_t)x.vi[v], (uint64_t)(x.vi[v] >> 63));
      if (d.off_min >= 0) atomicMax((unsigned long long*)(e + d.off_min), (unsigned long long)enc_min_i(x.vi[v]));
      if (d.off_max >= 0) atomicMax((unsigned long long*)(e + d.off_max), (unsigned long long)enc_max_i(x.vi[v]));
    }
  }
}

// Warp-level run combining before the HBM atomics (many-groups tier).  Lanes own
// consecutive rows, so runs of equal keys (clustered inputs such as lineitem
// ordered by orderkey, or hot keys) are contiguous lane ranges: one segmented
// shuffle reduction folds each run into its first lane, which alone touches the
// table.  Rows that are not eligible (slow values, the key ~0) take the per-row path.
template <int NV, bool F64>
__device__ __forceinline__ void glb_unit(const Plan& p, const RowIn<NV, F64>& x, int64_t r, int lane) {
  const bool ok = x.q && x.fast && x.key != ~0ULL;
  const unsigned okmask = __ballot_sync(0xffffffffu, ok);
  const uint64_t kprev = __shfl_up_sync(0xffffffffu, x.key, 1);
  const bool cont = ok && lane > 0 && ((okmask >> (lane - 1)) & 1u) && kprev == x.key;
  const unsigned contmask = __ballot_sync(0xffffffffu, cont);
  if (contmask == 0) {                   // no run in this unit (shuffled / high-cardinality): per row
    glb_row<NV, F64>(p, x, r);
    return;
  }
  if (x.q && !ok) glb_row<NV, F64>(p, x, r);
  const unsigned later = lane == 31 ? 0u : (~contmask & ~((2u << lane) - 1u));   // segment starts after me
  const int seg_end = later ? __ffs(later) - 2 : 31;
  uint32_t c = ok ? 1u : 0u;
  I128 si[F64 ? 1 : NV];
  double sd[F64 ? NV : 1], mnd[F64 ? NV : 1], mxd[F64 ? NV : 1];
  int64_t mni[F64 ? 1 : NV], mxi[F64 ? 1 : NV];
#pragma unroll
  for (int v = 0; v < NV; ++v) {
    if constexpr (F64) {
      sd[v] = ok ? x.vd[v] : 0.0;
      mnd[v] = x.vd[v];
      mxd[v] = x.vd[v];
    } else {
      si[v] = ok ? i128_from_i64(x.vi[v]) : I128{0, 0};
      mni[v] = x.vi[v];
      mxi[v] = x.vi[v];
    }
  }
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    const bool take = lane + o <= seg_end;
    const uint32_t cy = __shfl_down_sync(0xffffffffu, c, o);   // every lane shuffles; `take` selects
    if (take) c += cy;
#pragma unroll
    for (int v = 0; v < NV; ++v) {
      if (v >= p.nvals) break;
      const DevValue& d = p.vals[v];
      if constexpr (F64) {
        double y = __shfl_down_sync(0xffffffffu, sd[v], o);
        if (take) sd[v] += y;
        if (d.off_min >= 0) { double z = __shfl_down_sync(0xffffffffu, mnd[v], o); if (take) mnd[v] = fmin(mnd[v], z); }
        if (d.off_max >= 0) { double z = __shfl_down_sync(0xffffffffu, mxd[v], o); if (take) mxd[v] = fmax(mxd[v], z); }
      } else {
        if (d.off_sum >= 0) {
          I128 y;
          y.lo = __shfl_down_sync(0xffffffffu, si[v].lo, o);
          y.hi = __shfl_down_sync(0xffffffffu, si[v].hi, o);
          if (take) si[v] = i128_add(si[v], y);
        }
        if (d.off_min >= 0) {
          int64_t z = (int64_t)__shfl_down_sync(0xffffffffu, (long long)mni[v], o);
          if (take) mni[v] = min(mni[v], z);
        }
        if (d.off_max >= 0) {
          int64_t z = (int64_t)__shfl_down_sync(0xffffffffu, (long long)mxi[v], o);
          if (take) mxi[v] = max(mxi[v], z);
        }
      }
    }
  }
  if (!ok || cont) return;                // run heads only
  uint8_t* e = table_find_or_insert(p.table, p.mask, p.stride, x.key, p.status);
  if (!e) return;
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

template <int NV, bool F64, int U>
__global__ void __launch_bounds__(kFusedThreads) k_sga_glb(const __grid_constant__ Plan p) {
  const int lane = threadIdx.x & 31;
  constexpr int kTile = 32 * U;            // lane l owns rows base + 32u + l: consecutive rows across lanes
  const int64_t warp = (blockIdx.x * (int64_t)blockDim.x + threadIdx.x) >> 5;
  const int64_t nwarps = ((int64_t)gridDim.x * blockDim.x) >> 5;
  const int64_t ntiles = (p.n + kTile - 1) / kTile;
  for (int64_t t = warp; t < ntiles; t += nwarps) {
    const int64_t base = t * kTile;
    RowIn<NV, F64> x[U];
#pragma unroll
    for (int u = 0; u < U; ++u) eval_row_scalar<NV, F64>(p, base + 32 * u + lane, x[u]);
#pragma unroll
    for (int u = 0; u < U; ++u) {
      const int64_t r = base + 32 * u + lane;
      if (p.bitmap_out) {
        const uint32_t w = __ballot_sync(0xffffffffu, x[u].q);
        const int64_t wi = r >> 5;
        if (lane == 0 && wi < ((p.n + 31) >> 5)) p.bitmap_out[wi] = w;
      }
      glb_unit<NV, F64>(p, x[u], r, lane);
    }
  }
}

// ------------------------------------------------------------------ dispatch
constexpr int kUnits = 2;
constexpr int kGlbUnits = 4;

static size_t reg_smem(const Plan& p) {
  return (size_t)kRegSlots * p.priv_rec * kFusedThreads + (size_t)p.smem_cap * p.cta_stride;
}

template <int NV, bool F64>
static cudaError_t launch_reg_nv(const Plan& p, int grid, cudaStream_t s) {
  const size_t smem = reg_smem(p);
  cudaError_t e = cudaFuncSetAttribute(k_sga_reg<NV, F64, kUnits>, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                       (int)smem);
  if (e != cudaSuccess) return e;
  count_launch();
  k_sga_reg<NV, F64, kUnits><<<grid, kFusedThreads, smem, s>>>(p);
  return cudaGetLastError();
}

template <bool F64>
static cudaError_t launch_reg_f(const Plan& p, int grid, cudaStream_t s) {
  if (p.nvals <= 1) return launch_reg_nv<1, F64>(p, grid, s);
  if (p.nvals <= 2) return launch_reg_nv<2, F64>(p, grid, s);
  if (p.nvals <= 4) return launch_reg_nv<4, F64>(p, grid, s);
  return launch_reg_nv<6, F64>(p, grid, s);
}

template <bool F64>
static cudaError_t launch_glb_f(const Plan& p, int grid, cudaStream_t s) {
  count_launch();
  if (p.nvals <= 1) k_sga_glb<1, F64, kGlbUnits><<<grid, kFusedThreads, 0, s>>>(p);
  else if (p.nvals <= 2) k_sga_glb<2, F64, kGlbUnits><<<grid, kFusedThreads, 0, s>>>(p);
  else if (p.nvals <= 4) k_sga_glb<4, F64, kGlbUnits><<<grid, kFusedThreads, 0, s>>>(p);
  else k_sga_glb<6, F64, kGlbUnits><<<grid, kFusedThreads, 0, s>>>(p);
  return cudaGetLastError();
}

int reg_tier_slots() { return kRegSlots; }

template <int NV, bool F64>
static const void* reg_kernel_ptr() { return (const void*)k_sga_reg<NV, F64, kUnits>; }
template <int NV, bool F64>
static const void* glb_kernel_ptr() { return (const void*)k_sga_glb<NV, F64, kGlbUnits>; }

// Resident CTAs per SM of the instantiation launch_fused would pick (persistent grid sizing).
int fused_blocks_per_sm(const Plan& p, bool reg_tier, bool values_f64) {
  const int nv = p.nvals <= 1 ? 1 : (p.nvals <= 2 ? 2 : (p.nvals <= 4 ? 4 : 6));
  const void* fn;
  if (reg_tier) {
    if (values_f64) fn = nv == 1 ? reg_kernel_ptr<1, true>() : nv == 2 ? reg_kernel_ptr<2, true>() : nv == 4 ? reg_kernel_ptr<4, true>() : reg_kernel_ptr<6, true>();
    else fn = nv == 1 ? reg_kernel_ptr<1, false>() : nv == 2 ? reg_kernel_ptr<2, false>() : nv == 4 ? reg_kernel_ptr<4, false>() : reg_kernel_ptr<6, false>();
    cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)reg_smem(p));
  } else {
    if (values_f64) fn = nv == 1 ? glb_kernel_ptr<1, true>() : nv == 2 ? glb_kernel_ptr<2, true>() : nv == 4 ? glb_kernel_ptr<4, true>() : glb_kernel_ptr<6, true>();
    else fn = nv == 1 ? glb_kernel_ptr<1, false>() : nv == 2 ? glb_kernel_ptr<2, false>() : nv == 4 ? glb_kernel_ptr<4, false>() : glb_kernel_ptr<6, false>();
  }
  int nb = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&nb, fn, kFusedThreads, reg_tier ? reg_smem(p) : 0) != cudaSuccess ||
      nb < 1)
    nb = 1;
  return nb;
}

// values_f64: all value expressions are fp64 (mixed int/fp64 plans use the
// integer kernels, whose slow path handles fp64 values exactly too).
cudaError_t launch_fused(const Plan& p, bool reg_tier, bool values_f64, int grid, cudaStream_t s) {
  if (p.n == 0) return cudaSuccess;
  int64_t tiles = (p.n + 64 * kUnits - 1) / (64 * kUnits);
  int64_t g = (tiles + (kFusedThreads / 32) - 1) / (kFusedThreads / 32);
  if (g > grid) g = grid;
  if (reg_tier) return values_f64 ? launch_reg_f<true>(p, (int)g, s) : launch_reg_f<false>(p, (int)g, s);
  return values_f64 ? launch_glb_f<true>(p, (int)g, s) : launch_glb_f<false>(p, (int)g, s);
}

}  // namespace ocl
