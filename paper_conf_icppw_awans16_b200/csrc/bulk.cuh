// bulk.cuh — TMA 1-D bulk copies (cp.async.bulk) and mbarrier helpers, raw PTX
// for sm_100a. Used to prefetch the next array of a warp into shared memory
// while the current one is being sorted.
#pragma once
#include <cstdint>

namespace gas {

__device__ __forceinline__ uint32_t smem_u32(const void* p) {
  return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}

__device__ __forceinline__ void mbar_init(uint64_t* bar, uint32_t count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count) : "memory");
}

// Make mbarrier initialisation visible to the async (TMA) proxy.
__device__ __forceinline__ void fence_mbar_init() {
  asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
}

// Order this thread's earlier generic-proxy shared-memory accesses before
// later async-proxy (bulk copy) accesses to the same buffer.
__device__ __forceinline__ void fence_proxy_async_smem() {
  asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
}

__device__ __forceinline__ void mbar_arrive_expect_tx(uint64_t* bar, uint32_t bytes) {
  asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes)
               : "memory");
}

// Global -> shared bulk copy; completion is signalled on `bar` as tx bytes.
// dst, src 16-byte aligned; bytes a multiple of 16.
__device__ __forceinline__ void bulk_g2s(void* dst, const void* src, uint32_t bytes, uint64_t* bar) {
  asm volatile(
      "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
          smem_u32(dst)),
      "l"(src), "r"(bytes), "r"(smem_u32(bar))
      : "memory");
}

__device__ __forceinline__ void mbar_wait_parity(uint64_t* bar, uint32_t parity) {
  const uint32_t a = smem_u32(bar);
  uint32_t done;
  do {
    asm volatile(
        "{\n\t.reg .pred p;\n\t"
        "mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n\t"
        "selp.u32 %0, 1, 0, p;\n\t}"
        : "=r"(done)
        : "r"(a), "r"(parity)
        : "memory");
  } while (!done);
}

// One lane (elect.sync: the lowest active lane) issues the bulk operation;
// no branch, so no BSSY / BSYNC around it (GAS_BK_ELECT). The same lane always
// wins while the warp is converged, which the bulk-group waits rely on.
#ifndef GAS_BK_ELECT
#define GAS_BK_ELECT 1
#endif
__device__ __forceinline__ void bulk_prefetch_elect(bool p, const void* g, uint32_t bytes) {
  asm volatile("{\n\t.reg .pred e, q;\n\telect.sync _|e, 0xffffffff;\n\tsetp.ne.and.u32 q, %2, 0, e;\n\t"
               "@q cp.async.bulk.prefetch.L2.global [%0], %1;\n\t}"
               ::"l"(g), "r"(bytes), "r"((uint32_t)p) : "memory");
}
__device__ __forceinline__ void bulk_store_elect(void* g, uint32_t sa, uint32_t bytes) {
  asm volatile("{\n\t.reg .pred e;\n\telect.sync _|e, 0xffffffff;\n\t"
               "@e cp.async.bulk.global.shared::cta.bulk_group [%0], [%1], %2;\n\t@e cp.async.bulk.commit_group;\n\t}"
               ::"l"(g), "r"(sa), "r"(bytes) : "memory");
}
// prefetch_l2 (the 16-byte-aligned cover of [p, p + words)) issued by one elected lane when `pred`
__device__ __forceinline__ void prefetch_l2_elect(bool pred, const uint32_t* p, int64_t words) {
  const uintptr_t a = reinterpret_cast<uintptr_t>(p) & ~(uintptr_t)15;
  const uintptr_t e = (reinterpret_cast<uintptr_t>(p + words) + 15) & ~(uintptr_t)15;
  bulk_prefetch_elect(pred, reinterpret_cast<const void*>(a), (uint32_t)(e - a));
}
__device__ __forceinline__ void bulk_wait_read_elect() {
  asm volatile("{\n\t.reg .pred e;\n\telect.sync _|e, 0xffffffff;\n\t@e cp.async.bulk.wait_group.read 0;\n\t}" ::: "memory");
}

}  // namespace gas
