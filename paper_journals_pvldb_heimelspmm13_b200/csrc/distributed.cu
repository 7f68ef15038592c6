// distributed.cu — the multi-GPU exchange of partial group tables.
//
// The paper runs one device at a time; multi-device execution is its stated future
// work (§6).  Here each rank aggregates its row shard into a partial
// table, and the library itself exchanges the partials over NCCL on the call's stream
// (no host synchronisation, so a whole distributed call is CUDA-graph capturable):
//
//  * allgather (ocl_sga_args.distributed = 1): every rank sends its partial table padded
//    to the partial capacity plus a 16-byte header {rows, status}; every rank merges all P
//    tables -> replicated result.  Q1 (4 groups): ~1.5 KB per rank, latency-bound.
//  * all-to-all (distributed = 2): every partial row goes to the rank owning its key's
//    hash partition, d = ((fmix64(key) & 0xFFFFFFFF) * P) >> 32 (as ocl_route_partials),
//    in fixed-size blocks of B rows per destination (so the NCCL send sizes are known on
//    the host); the header carries the P per-destination row counts and the status.
//    Each rank merges what it receives -> its hash partition of the groups.  This is the
//    paper's "partitioning instead of one global hash table" (L793-796) across devices.
//
// Overflow protocol (the paper's restart, L523-527): every rank sees every header, so all
// ranks take the same decision — if any partial overflowed (status != 0, rows > capacity,
// or a destination block > B) the merge is skipped everywhere, dev_status =
// OCL_ERR_CAPACITY on every rank, and ocl_select_group_aggregate_sync re-runs all ranks in
// lockstep with a larger table.
//
// NCCL is loaded at run time (dlopen "libnccl.so.2": in a PyTorch process that is the
// library torch already loaded), so libocelot_b200.so has no link-time NCCL dependency.
#include <dlfcn.h>
#include <stdio.h>
#include <string.h>

#include <mutex>

#include <nccl.h>

#include "launch.cuh"

namespace ocl {

namespace {

struct NcclApi {
  bool ok = false;
  decltype(&ncclGetUniqueId) GetUniqueId = nullptr;
  decltype(&ncclCommInitRank) CommInitRank = nullptr;
  decltype(&ncclCommDestroy) CommDestroy = nullptr;
  decltype(&ncclAllGather) AllGather = nullptr;
  decltype(&ncclSend) Send = nullptr;
  decltype(&ncclRecv) Recv = nullptr;
  decltype(&ncclGroupStart) GroupStart = nullptr;
  decltype(&ncclGroupEnd) GroupEnd = nullptr;
  decltype(&ncclGetErrorString) GetErrorString = nullptr;
};

std::mutex g_nccl_mu;
NcclApi g_nccl;

int nccl_load(char* err, size_t errlen) {
  std::lock_guard<std::mutex> lk(g_nccl_mu);
  if (g_nccl.ok) return 0;
  void* h = dlopen("libnccl.so.2", RTLD_NOW | RTLD_GLOBAL);
  if (!h) h = dlopen("libnccl.so", RTLD_NOW | RTLD_GLOBAL);
  if (!h) {
    snprintf(err, errlen, "NCCL not loadable: %s", dlerror());
    return 1;
  }
  NcclApi a;
#define OCL_SYM(field, name)                                                   \
  a.field = (decltype(a.field))dlsym(h, name);                                 \
  if (!a.field) {                                                              \
    snprintf(err, errlen, "NCCL symbol %s missing", name);                     \
    return 1;                                                                  \
  }
  OCL_SYM(GetUniqueId, "ncclGetUniqueId");
  OCL_SYM(CommInitRank, "ncclCommInitRank");
  OCL_SYM(CommDestroy, "ncclCommDestroy");
  OCL_SYM(AllGather, "ncclAllGather");
  OCL_SYM(Send, "ncclSend");
  OCL_SYM(Recv, "ncclRecv");
  OCL_SYM(GroupStart, "ncclGroupStart");
  OCL_SYM(GroupEnd, "ncclGroupEnd");
  OCL_SYM(GetErrorString, "ncclGetErrorString");
#undef OCL_SYM
  a.ok = true;
  g_nccl = a;
  return 0;
}

int nccl_check(ncclResult_t r, const char* what, char* err, size_t errlen) {
  if (r == ncclSuccess) return 0;
  snprintf(err, errlen, "%s: %s", what, g_nccl.GetErrorString ? g_nccl.GetErrorString(r) : "NCCL error");
  return 1;
}

}  // namespace

int nccl_unique_id(void* id128, char* err, size_t errlen) {
  if (nccl_load(err, errlen)) return 1;
  static_assert(sizeof(ncclUniqueId) == 128, "ncclUniqueId is 128 bytes");
  ncclUniqueId id;
  if (nccl_check(g_nccl.GetUniqueId(&id), "ncclGetUniqueId", err, errlen)) return 1;
  memcpy(id128, &id, sizeof(id));
  return 0;
}

int nccl_comm_init(void** comm, const void* id128, int rank, int nranks, char* err, size_t errlen) {
  if (nccl_load(err, errlen)) return 1;
  ncclUniqueId id;
  memcpy(&id, id128, sizeof(id));
  ncclComm_t c = nullptr;
  if (nccl_check(g_nccl.CommInitRank(&c, nranks, id, rank), "ncclCommInitRank", err, errlen)) return 1;
  *comm = c;
  return 0;
}

void nccl_comm_destroy(void* comm) {
  if (comm && g_nccl.ok) g_nccl.CommDestroy((ncclComm_t)comm);
}

int nccl_allgather2(const void* a, void* a_all, size_t a_bytes, const void* b, void* b_all, size_t b_bytes,
                    void* comm, cudaStream_t s, char* err, size_t errlen) {
  ncclComm_t c = (ncclComm_t)comm;
  if (nccl_check(g_nccl.GroupStart(), "ncclGroupStart", err, errlen)) return 1;
  ncclResult_t r = g_nccl.AllGather(a, a_all, a_bytes, ncclUint8, c, s);
  if (r == ncclSuccess && b_bytes) r = g_nccl.AllGather(b, b_all, b_bytes, ncclUint8, c, s);
  ncclResult_t r2 = g_nccl.GroupEnd();
  if (nccl_check(r, "ncclAllGather", err, errlen)) return 1;
  return nccl_check(r2, "ncclGroupEnd", err, errlen);
}

int nccl_alltoall_blocks(const void* hdr, void* hdr_all, size_t hdr_bytes, const void* send, void* recv,
                         size_t block_bytes, int nranks, void* comm, cudaStream_t s, char* err, size_t errlen) {
  ncclComm_t c = (ncclComm_t)comm;
  if (nccl_check(g_nccl.GroupStart(), "ncclGroupStart", err, errlen)) return 1;
  ncclResult_t r = g_nccl.AllGather(hdr, hdr_all, hdr_bytes, ncclUint8, c, s);
  for (int p = 0; p < nranks && r == ncclSuccess && block_bytes; ++p) {
    r = g_nccl.Send((const uint8_t*)send + (size_t)p * block_bytes, block_bytes, ncclUint8, p, c, s);
    if (r == ncclSuccess) r = g_nccl.Recv((uint8_t*)recv + (size_t)p * block_bytes, block_bytes, ncclUint8, p, c, s);
  }
  ncclResult_t r2 = g_nccl.GroupEnd();
  if (nccl_check(r, "ncclAllGather/ncclSend/ncclRecv", err, errlen)) return 1;
  return nccl_check(r2, "ncclGroupEnd", err, errlen);
}

// ------------------------------------------------------------------ kernels
// Headers of all ranks: hdr_all[p * W + w], W = hdr_words; words 0..W-2 are row counts
// (per destination for the all-to-all, one word for the allgather), word W-1 the rank's
// partial status.  counts_out[p] = rows this rank merges from rank p (column `col`);
// any overflow anywhere -> every count 0 and *status = OCL_ERR_CAPACITY (same decision
// on every rank: every rank reads the same headers).
// report = 1 (launched after the finalisation): on overflow, *ngroups_out = the largest
// partial row count of any rank (a lower bound on G: > out_capacity means the result cannot
// fit; otherwise a table overflowed and a restart with a larger table can succeed).
__global__ void k_dist_headers(const int64_t* hdr_all, int32_t nparts, int32_t W, int32_t col, int64_t cap,
                               int64_t* counts_out, int32_t* status, int32_t report, int64_t* ngroups_out) {
  __shared__ int bad;
  __shared__ unsigned long long gmax;
  if (threadIdx.x == 0) {
    bad = 0;
    gmax = 0;
  }
  __syncthreads();
  int my_bad = 0;
  for (int i = threadIdx.x; i < nparts * W; i += blockDim.x) {
    const int64_t x = hdr_all[i];
    const int w = i % W;
    if (w == W - 1 ? x != 0 : (x < 0 || x > cap)) my_bad = 1;
  }
  if (my_bad) atomicOr(&bad, 1);
  __syncthreads();
  if (report) {
    if (!bad) return;
    for (int p = threadIdx.x; p < nparts; p += blockDim.x) {
      long long g = 0;
      for (int w = 0; w < W - 1; ++w) g += hdr_all[(int64_t)p * W + w];
      atomicMax(&gmax, (unsigned long long)(g < 0 ? 0 : g));
    }
    __syncthreads();
    if (threadIdx.x == 0) *ngroups_out = (int64_t)gmax;
    return;
  }
  for (int p = threadIdx.x; p < nparts; p += blockDim.x) counts_out[p] = bad ? 0 : hdr_all[(int64_t)p * W + col];
  if (threadIdx.x == 0 && bad && status) atomicCAS(status, 0, (int32_t)OCL_ERR_CAPACITY);
}

__device__ __forceinline__ uint32_t dist_route(uint64_t key, uint32_t nparts) {
  return (uint32_t)(((fmix64(key) & 0xFFFFFFFFULL) * nparts) >> 32);
}

// Route partial rows into fixed blocks: destination d's rows at out + (d * block_rows +
// slot) * row_bytes; counts[d] = rows destined to d (may exceed block_rows: overflow,
// detected by k_dist_headers on every rank).
__global__ void k_route_blocks(const uint8_t* rows, const int64_t* nrows_dev, int64_t max_rows, int32_t row_bytes,
                               uint32_t nparts, int64_t block_rows, uint8_t* out, unsigned long long* counts) {
  const int64_t n = min(*nrows_dev, max_rows);
  const int words = row_bytes / 8;
  for (int64_t r = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; r < n; r += (int64_t)gridDim.x * blockDim.x) {
    const uint64_t* src = (const uint64_t*)(rows + r * row_bytes);
    const uint32_t d = dist_route(src[0], nparts);
    const unsigned long long slot = atomicAdd(&counts[d], 1ULL);
    if ((int64_t)slot >= block_rows) continue;
    uint64_t* dst = (uint64_t*)(out + ((int64_t)d * block_rows + (int64_t)slot) * row_bytes);
    for (int w = 0; w < words; ++w) dst[w] = src[w];
  }
}

cudaError_t launch_dist_headers(const int64_t* hdr_all, int32_t nparts, int32_t hdr_words, int32_t col, int64_t cap,
                                int64_t* counts_out, int32_t* status, int32_t report, int64_t* ngroups_out,
                                cudaStream_t s) {
  count_launch();
  k_dist_headers<<<1, 256, 0, s>>>(hdr_all, nparts, hdr_words, col, cap, counts_out, status, report, ngroups_out);
  return cudaGetLastError();
}

cudaError_t launch_route_blocks(const void* rows, const int64_t* nrows_dev, int64_t max_rows, int32_t row_bytes,
                                int32_t nparts, int64_t block_rows, void* out, int64_t* counts, int sms,
                                cudaStream_t s) {
  if (max_rows == 0) return cudaSuccess;
  int64_t grid = (max_rows + 255) / 256;
  if (grid > (int64_t)sms * 4) grid = (int64_t)sms * 4;
  count_launch();
  k_route_blocks<<<(int)grid, 256, 0, s>>>((const uint8_t*)rows, nrows_dev, max_rows, row_bytes, (uint32_t)nparts,
                                           block_rows, (uint8_t*)out, (unsigned long long*)counts);
  return cudaGetLastError();
}

}  // namespace ocl
