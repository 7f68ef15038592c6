// launch.cuh — host-side launcher interface between abi.cu and the kernel files.
#pragma once

#include <atomic>

#include "common.cuh"

namespace ocl {
// Kernel launches issued by this library (evidence for the benchmark's gpu_launches).
extern std::atomic<unsigned long long> g_launches;
inline void count_launch(unsigned long long k = 1) { g_launches.fetch_add(k, std::memory_order_relaxed); }

// Per-device cache of a kernel's launch setup (dynamic shared-memory attribute set,
// resident CTAs per SM).  Attributes and occupancy belong to a device, not to the
// process: one process may drive several GPUs.  Racing initialisations compute the
// same value, so relaxed atomics suffice.
constexpr int kMaxDevices = 64;
struct DevCache {
  std::atomic<int> v[kMaxDevices];
  DevCache() {
    for (auto& x : v) x.store(-1, std::memory_order_relaxed);
  }
  // value for the current device, computing it with f() on first use
  template <class F>
  int get(F f) {
    int d = 0;
    if (cudaGetDevice(&d) != cudaSuccess || d < 0 || d >= kMaxDevices) return f();
    int x = v[d].load(std::memory_order_relaxed);
    if (x < 0) {
      x = f();
      v[d].store(x, std::memory_order_relaxed);
    }
    return x;
  }
};

struct SelParams {
  const void* col;
  int64_t n;
  int32_t dtype;
  int32_t is_f64;
  int32_t anti;
  int32_t vec_ok;      // column pointer 16-byte aligned
  int64_t lo, hi;      // normalised inclusive bounds
  double flo, fhi;
  uint32_t* out;
  int32_t lo32, hi32;  // bounds clamped to the column's range (empty range: lo32 > hi32); set by the launcher
};
struct EmitArgs {
  int32_t kind;
  FinPlan fin;
  int64_t* keys_out;
  int64_t out_capacity;
  uint8_t* partial_out;
  int32_t* status;
};
enum EmitKind : int32_t { EMIT_FINAL = 0, EMIT_PARTIAL = 2 };

cudaError_t launch_select_bitmap(const SelParams& p, int grid, cudaStream_t s);
cudaError_t launch_bitmap_combine(int op, const uint32_t* a, const uint32_t* b, uint32_t* out, int64_t n, int grid,
                                  cudaStream_t s);
size_t prefix_compact_ws_bytes(int64_t n);
cudaError_t launch_prefix_compact(const uint32_t* bitmap, int64_t n, uint32_t* oids, int64_t* m_out, void* ws,
                                  int grid, cudaStream_t s);
size_t emit_ws_bytes(int grid);
cudaError_t launch_emit(uint8_t* table, uint64_t cap, int32_t stride, const EmitArgs& a, int64_t* ngroups_out,
                        int64_t out_capacity, int32_t* status, bool sorted, void* ws, int grid, cudaStream_t s);
bool sorted_emit_supported(uint64_t cap);
cudaError_t launch_finalize_dense(const uint8_t* table, int32_t stride, const int64_t* ngroups, int64_t max_groups,
                                  const FinPlan& f, int grid, cudaStream_t s);
cudaError_t launch_group_build(const Plan& p, int32_t* gid_out, int64_t max_rows, int64_t* ngroups,
                               int64_t* keys_out, int64_t out_capacity, int grid, cudaStream_t s);
cudaError_t launch_gather(const void* col, int32_t width, const uint32_t* oids, const int64_t* m_dev, int64_t max_m,
                          void* out, int grid, cudaStream_t s);
cudaError_t launch_merge_partials(const uint8_t* partials, int32_t nparts, int64_t part_capacity,
                                  const int64_t* part_counts, const FinPlan& f, uint8_t* table, uint64_t mask,
                                  int32_t* status, int grid, cudaStream_t s);
cudaError_t launch_group_aggregate(const Plan& p, int64_t max_rows, const int64_t* ngroups_dev, int64_t max_groups,
                                   bool values_f64, int sms, cudaStream_t s);
// Fused select -> group -> aggregate kernel (fused.cu).  mode 0: static shape if one
// matches the plan, else dynamic; 1: dynamic shape only; 2: HBM-only kernel.
cudaError_t launch_fused(const Plan& p, int mode, bool values_f64, int sms, cudaStream_t s, int* kind);
int reg_tier_slots();
const char* fused_kernel_name(int kind);
// Proven few-group Q1 kernel (fused_spec.cu) used while the unified kernel is tuned.
bool launch_fused_spec(const Plan& g, int sms, cudaStream_t s, cudaError_t* err, int* kind);
// Whether a plan-signature kernel takes this group-by plan (the planner keeps the one-pass tier).
bool spec_takes(const Plan& g);
int32_t spec_mm_check(int64_t expected_groups);
int32_t spec_sparse_pct(int64_t n);
int32_t spec_twin_pct(int32_t pct, bool has_pred, bool private_tier);
// CTA-table tier of the signature kernels (fused_spec.cu): consumer threads T, rows per
// stage R, stages NS, 2^hb slots x nrep tables, MIN / MAX read-before-atomic
struct TabPolicy {
  int T, R, NS;
  uint32_t hb, nrep;
  int32_t mm_check;
};
bool tab_policy(int64_t expected_groups, size_t slot_bytes, size_t row_bytes, TabPolicy* tp);
// The signature kernels compiled at run time for a plan no compiled-in signature matches (jit.cu).
bool launch_fused_jit(const Plan& g, int sms, cudaStream_t s, cudaError_t* err, int* kind);
// High-cardinality tier (partition.cu): hash-partitioned two-pass aggregation.
bool part_eligible(const Plan& p);
int part_bits_for(int64_t expected_groups, int64_t n);
size_t part_ws_bytes(const Plan& p, int pbits, int sms);
// ea != NULL: emit the output rows (final or partial) directly, count -> *count_out, *emitted = true
// (else the caller emits from the HBM table).
cudaError_t launch_partitioned(const Plan& p, int pbits, void* ws, int sms, cudaStream_t s, int* kind,
                               const EmitArgs* ea = nullptr, int64_t* count_out = nullptr, int64_t out_capacity = 0,
                               bool* emitted = nullptr);
// Hash routing of partial rows for the all-to-all merge (exchange.cu, NEXT-2).
size_t route_ws_bytes(int32_t nparts);
int route_max_parts();
cudaError_t launch_route(const void* rows, const int64_t* nrows_dev, int64_t max_rows, int32_t row_bytes,
                         int32_t nparts, void* out, int64_t* part_counts, void* ws, int sms, cudaStream_t s);
// Multi-GPU exchange over NCCL (distributed.cu; NCCL loaded at run time).  The int
// functions return 0 on success, else 1 with a message in err.
int nccl_unique_id(void* id128, char* err, size_t errlen);
int nccl_comm_init(void** comm, const void* id128, int rank, int nranks, char* err, size_t errlen);
void nccl_comm_destroy(void* comm);
int nccl_allgather2(const void* a, void* a_all, size_t a_bytes, const void* b, void* b_all, size_t b_bytes,
                    void* comm, cudaStream_t s, char* err, size_t errlen);
int nccl_alltoall_blocks(const void* hdr, void* hdr_all, size_t hdr_bytes, const void* send, void* recv,
                         size_t block_bytes, int nranks, void* comm, cudaStream_t s, char* err, size_t errlen);
cudaError_t launch_dist_headers(const int64_t* hdr_all, int32_t nparts, int32_t hdr_words, int32_t col, int64_t cap,
                                int64_t* counts_out, int32_t* status, int32_t report, int64_t* ngroups_out,
                                cudaStream_t s);
cudaError_t launch_route_blocks(const void* rows, const int64_t* nrows_dev, int64_t max_rows, int32_t row_bytes,
                                int32_t nparts, int64_t block_rows, void* out, int64_t* counts, int sms,
                                cudaStream_t s);
// Equi hash join (join.cu).
size_t join_build_ws_bytes(int64_t n_build);
size_t join_probe_ws_bytes(int64_t max_rows);
cudaError_t launch_join_build(const DevKey& bk, int64_t n_build, void* ws, int32_t* status, int sms, cudaStream_t s);
cudaError_t launch_join_probe(const void* build_ws, int64_t n_build, const DevKey& pk, const uint32_t* oids,
                              const int64_t* m_dev, int64_t max_rows, bool pk_build, uint32_t* out_probe,
                              uint32_t* out_build, int64_t out_capacity, int64_t* nout, int32_t* status, void* ws,
                              int sms, cudaStream_t s);
// The paper's hashing scheme for the ablation (hashpaper.cu).
size_t hp_ws_bytes(int64_t max_rows, int64_t expected);
cudaError_t launch_group_build_paper(const Plan& p, int64_t expected, int32_t* gid_out, int64_t* keys_out,
                                     int64_t out_capacity, int64_t* ngroups, void* ws, int sms, cudaStream_t s);
// LSD radix sort of packed keys (radix.cu).
size_t radix_ws_bytes(int64_t n, bool val, bool row);
cudaError_t launch_radix(const Plan& p, const uint64_t* vcol, uint64_t* kout, uint64_t* vout, uint32_t* rout,
                         void* ws, int sms, cudaStream_t s);
// Sorted-input GROUP BY (sorted.cu).
size_t sorted_ws_bytes(const Plan& p);
cudaError_t launch_sorted(const Plan& p, const FinPlan& fin, bool values_f64, void* ws, int32_t* status,
                          int64_t* ngroups_out, int64_t out_capacity, int sms, cudaStream_t s, int* kind,
                          uint8_t* partial_out = nullptr);
size_t group_build_sorted_ws_bytes(int64_t max_rows);
cudaError_t launch_group_build_sorted(const Plan& p, int32_t* gid_out, int64_t* keys_out, int64_t out_capacity,
                                      int64_t* ngroups, void* ws, int sms, cudaStream_t s);
}  // namespace ocl
