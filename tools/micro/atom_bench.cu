// Microbenchmark: random global RED / probe+RED throughput vs table size (design input for
// the high-cardinality tier).  nvcc -gencode arch=compute_100a,code=sm_100a -O3
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>
__device__ __forceinline__ uint64_t fmix64(uint64_t k) {
  k ^= k >> 33; k *= 0xff51afd7ed558ccdULL; k ^= k >> 33; k *= 0xc4ceb9fe1a85ec53ULL; k ^= k >> 33; return k;
}
// mode 0: 4 REDs per row into a random 64-B entry; 1: probe load of the key word then 4 REDs
// mode 2: 1 RED per row; 3: 2 rows per thread in flight probe+RED
__global__ void k_red(uint64_t* tab, uint64_t mask, int64_t n, int mode) {
  int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x, st = (int64_t)gridDim.x * blockDim.x;
  for (; i < n; i += st) {
    uint64_t h = fmix64((uint64_t)i) & mask;
    uint64_t* e = tab + h * 8;
    if (mode == 1) {
      uint64_t k = *(volatile uint64_t*)e;
      if (k == 12345) continue;
    }
    atomicAdd((unsigned long long*)(e + 1), 1ULL);
    if (mode != 2) {
      atomicAdd((unsigned long long*)(e + 2), (unsigned long long)i);
      atomicMax((unsigned long long*)(e + 3), (unsigned long long)i);
      atomicMax((unsigned long long*)(e + 4), (unsigned long long)~i);
    }
  }
}
__global__ void k_stream(const int4* a, int64_t n4, int4* out) {
  int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x, st = (int64_t)gridDim.x * blockDim.x;
  int4 acc = make_int4(0,0,0,0);
  for (; i < n4; i += st) { int4 v = __ldg(a + i); acc.x ^= v.x; acc.y ^= v.y; acc.z ^= v.z; acc.w ^= v.w; }
  if (acc.x == 0x7fffffff) out[0] = acc;
}
int main() {
  const int64_t n = 1LL << 28;
  uint64_t* tab; cudaMalloc(&tab, (2ULL << 30) + 64);
  cudaEvent_t a, b; cudaEventCreate(&a); cudaEventCreate(&b);
  int sms; cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  for (int mode = 0; mode < 3; ++mode)
  for (uint64_t slots : {1ULL << 10, 1ULL << 16, 1ULL << 20, 1ULL << 22, 1ULL << 24, 1ULL << 25}) {
    cudaMemset(tab, 0, slots * 64);
    k_red<<<sms * 8, 256>>>(tab, slots - 1, n, mode);
    cudaEventRecord(a);
    k_red<<<sms * 8, 256>>>(tab, slots - 1, n, mode);
    cudaEventRecord(b); cudaEventSynchronize(b);
    float ms; cudaEventElapsedTime(&ms, a, b);
    printf("mode %d table %8.1f MB  %.3f ms  %.2f G rows/s  %.1f G atom/s\n", mode, slots * 64 / 1e6, ms,
           n / ms / 1e6, n * (mode == 2 ? 1 : 4) / ms / 1e6);
  }
  int4* buf; cudaMalloc(&buf, 8ULL << 30);
  cudaMemset(buf, 1, 8ULL << 30);
  for (int rep = 0; rep < 3; ++rep) {
    cudaEventRecord(a);
    k_stream<<<sms * 8, 512>>>(buf, (8LL << 30) / 16, (int4*)tab);
    cudaEventRecord(b); cudaEventSynchronize(b);
    float ms; cudaEventElapsedTime(&ms, a, b);
    printf("stream read 8 GiB: %.3f ms  %.1f GB/s\n", ms, 8.0 * (1 << 30) / ms / 1e6);
  }
  printf("%s\n", cudaGetErrorString(cudaGetLastError()));
}
