// Microbenchmark: shared-memory atomic vs plain read-modify-write throughput on random
// addresses (design input for the partition-aggregate pass).
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>
__device__ __forceinline__ uint32_t mix32(uint32_t x) { x ^= x >> 16; x *= 0x7feb352dU; x ^= x >> 15; x *= 0x846ca68bU; x ^= x >> 16; return x; }
template <int MODE>
__global__ void k(uint32_t* out, int iters, uint32_t mask) {
  extern __shared__ uint32_t sm[];
  for (int i = threadIdx.x; i <= (int)mask + 64; i += blockDim.x) sm[i] = 0;
  __syncthreads();
  uint32_t s = blockIdx.x * blockDim.x + threadIdx.x;
  uint32_t w = threadIdx.x >> 5;
  for (int it = 0; it < iters; ++it) {
    uint32_t h = mix32(s + it * 0x9e3779b9u);
    uint32_t a = h & mask;
    if (MODE == 0) atomicAdd(&sm[a], 1u);                                       // 1 x ATOMS.ADD.32
    if (MODE == 1) { atomicAdd(&sm[a], 1u); atomicAdd(&sm[a ^ 1], h); atomicMax(&sm[a ^ 2], h); atomicMin(&sm[a ^ 3], h); }
    if (MODE == 2) atomicAdd((unsigned long long*)&sm[a & ~1u], (unsigned long long)h);  // 64-bit add
    if (MODE == 3) { sm[a] += 1u; }                                             // plain RMW (racy, timing only)
    if (MODE == 4) { uint4 v = *(uint4*)&sm[a & ~3u]; v.x += 1; v.y += h; v.z = max(v.z, h); v.w = min(v.w, h); *(uint4*)&sm[a & ~3u] = v; }
    if (MODE == 5) { unsigned m = __match_any_sync(0xffffffffu, a >> 4); if (__popc(m) > 1) sm[a] += 1; }
  }
  if (threadIdx.x == 0) out[blockIdx.x] = sm[w];
}
int main() {
  uint32_t* out; cudaMalloc(&out, 1 << 20);
  int sms; cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  cudaEvent_t a, b; cudaEventCreate(&a); cudaEventCreate(&b);
  const int iters = 4096;
  for (uint32_t words : {8192u, 32768u}) {
    size_t smem = (words + 64) * 4;
    auto run = [&](auto fn, const char* name, int ops) {
      cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
      for (int threads : {256, 1024}) {
        int nb = 0; cudaOccupancyMaxActiveBlocksPerMultiprocessor(&nb, fn, threads, smem);
        fn<<<sms * nb, threads, smem>>>(out, iters, words - 1);
        cudaEventRecord(a);
        fn<<<sms * nb, threads, smem>>>(out, iters, words - 1);
        cudaEventRecord(b); cudaEventSynchronize(b);
        float ms; cudaEventElapsedTime(&ms, a, b);
        double rows = (double)sms * nb * threads * iters;
        printf("%-28s smem %6u B  thr %4d x %d  %.3f ms  %.1f G rows/s  %.2f rows/clk/SM  (%d ops/row)\n", name,
               words * 4, threads, nb, ms, rows / ms / 1e6, rows / ms / 1e6 / sms / 1.965, ops);
      }
    };
    run(k<0>, "ATOMS.ADD u32", 1);
    run(k<1>, "ATOMS add,add,max,min u32", 4);
    run(k<2>, "ATOMS.ADD u64", 1);
    run(k<3>, "plain LDS+STS u32", 1);
    run(k<4>, "plain LDS.128+STS.128", 4);
    run(k<5>, "match_any", 1);
  }
  printf("%s\n", cudaGetErrorString(cudaGetLastError()));
}
