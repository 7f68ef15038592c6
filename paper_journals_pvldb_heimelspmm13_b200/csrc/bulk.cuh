// bulk.cuh — TMA bulk copies (cp.async.bulk, global -> shared) and mbarrier helpers
// for the streaming producer/consumer pipelines (sm_100a).  A producer thread arms a
// stage's "full" barrier with the byte count and issues one bulk copy per column; the
// copy engine completes the transaction on the barrier; consumer warps wait on it,
// read the rows from shared memory and release the stage on its "empty" barrier.
#pragma once

#include <stdint.h>

namespace ocl {

__device__ __forceinline__ uint32_t smem_u32(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }

__device__ __forceinline__ void mbar_init(uint64_t* bar, uint32_t count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count) : "memory");
}

__device__ __forceinline__ void mbar_fence_init() {
  asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
}

__device__ __forceinline__ void mbar_arrive_expect_tx(uint64_t* bar, uint32_t bytes) {
  asm volatile("mbarrier.arrive.expect_tx.release.cta.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes)
               : "memory");
}

__device__ __forceinline__ void mbar_arrive(uint64_t* bar) {
  asm volatile("mbarrier.arrive.release.cta.shared::cta.b64 _, [%0];" ::"r"(smem_u32(bar)) : "memory");
}

// Release a stage that this warp has finished READING with generic-proxy loads (LDS) so
// that the producer may overwrite it with async-proxy (TMA) writes.  A plain
// mbarrier.arrive is not enough on sm_100a: ptxas issues the SYNCS.ARRIVE without waiting
// for the warp's outstanding LDS (empty wait mask in the SASS control bits), so the next
// bulk copy can land before the loads have read the stage — rows of two chunks mixed
// (seen as rare wrong group counts, most often with a 1-stage ring).  The cross-proxy
// fence orders the warp's generic reads before the async-proxy writes that follow the
// barrier (PTX: fence.proxy.async is required between generic and async proxy accesses
// to the same shared memory); every lane fences its own loads, then lane 0 arrives.
__device__ __forceinline__ void mbar_release_reads(uint64_t* bar, int lane) {
  asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
  __syncwarp();
  if (lane == 0) mbar_arrive(bar);
}

__device__ __forceinline__ bool mbar_try_wait(uint64_t* bar, uint32_t parity) {
  uint32_t ok;
  asm volatile(
      "{\n\t.reg .pred p;\n\t"
      "mbarrier.try_wait.parity.acquire.cta.shared::cta.b64 p, [%1], %2;\n\t"
      "selp.u32 %0, 1, 0, p;\n\t}"
      : "=r"(ok)
      : "r"(smem_u32(bar)), "r"(parity)
      : "memory");
  return ok != 0;
}

__device__ __forceinline__ void mbar_wait(uint64_t* bar, uint32_t parity) {
  while (!mbar_try_wait(bar, parity)) {
  }
}

// try_wait with a suspend-time hint: the thread is suspended (not re-issued) until the
// phase completes or `ns` nanoseconds pass.
__device__ __forceinline__ bool mbar_try_wait_hint(uint64_t* bar, uint32_t parity, uint32_t ns) {
  uint32_t ok;
  asm volatile(
      "{\n\t.reg .pred p;\n\t"
      "mbarrier.try_wait.parity.acquire.cta.shared::cta.b64 p, [%1], %2, %3;\n\t"
      "selp.u32 %0, 1, 0, p;\n\t}"
      : "=r"(ok)
      : "r"(smem_u32(bar)), "r"(parity), "r"(ns)
      : "memory");
  return ok != 0;
}

// Wait strategies (mode): 0 spin on try_wait; 1 back off with __nanosleep between tries
// (a waiting warp stops taking issue slots from the warps that have work); 2 try_wait
// with a suspend-time hint.
__device__ __forceinline__ void mbar_wait_mode(uint64_t* bar, uint32_t parity, int mode) {
  if (mode == 1) {
    uint32_t ns = 32;
    while (!mbar_try_wait(bar, parity)) {
      __nanosleep(ns);
      if (ns < 512) ns <<= 1;
    }
  } else if (mode == 2) {
    while (!mbar_try_wait_hint(bar, parity, 100000)) {
    }
  } else {
    mbar_wait(bar, parity);
  }
}

// 1-D bulk copy of `bytes` (multiple of 16; both addresses 16-byte aligned) from global
// to this CTA's shared memory, completing `bytes` transactions on `bar`.  Streamed
// input is read once: evict-first keeps it from displacing reusable lines in L2.
__device__ __forceinline__ void bulk_g2s(void* dst, const void* src, uint32_t bytes, uint64_t* bar, uint64_t policy) {
  asm volatile(
      "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes.L2::cache_hint [%0], [%1], %2, [%3], %4;" ::"r"(
          smem_u32(dst)),
      "l"(src), "r"(bytes), "r"(smem_u32(bar)), "l"(policy)
      : "memory");
}

__device__ __forceinline__ uint64_t policy_evict_first() {
  uint64_t pol;
  asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(pol));
  return pol;
}

}  // namespace ocl
