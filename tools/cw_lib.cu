// Experiment library for csrc/cw1024.cuh (built as its own .so so that its
// CUDA runtime and kernels do not collide with libgas.so's). See cw_exp.cu.
#include <cstdint>
#include <cuda_runtime.h>
#include "../paper_conf_icppw_awans16_b200/csrc/sort1024.cuh"

namespace gas {
// Stand-alone kernel (experiments, tools/cw_lib.cu): every array through
// cw_sort_warp. 16-byte-aligned rows, 512 < n <= 1024, 8 KB of shared memory per warp.
__global__ void __launch_bounds__(kCwBlock, 1)
    k_fixed_cw1024(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one, unsigned long long* stats) {
  extern __shared__ __align__(16) uint4 cw_smem[];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const uint32_t cnt_sa = (uint32_t)__cvta_generic_to_shared(cw_smem) + warp * kCwWarpBytes;
  const uint32_t buf_sa = cnt_sa + kCwCntBytes;
  uint32_t* const buf_ptr =
      reinterpret_cast<uint32_t*>(reinterpret_cast<unsigned char*>(cw_smem) + warp * kCwWarpBytes + kCwCntBytes);
  const int nc = n >> 2;
  const int64_t nwarps = (int64_t)gridDim.x * (kCwBlock / 32);
  unsigned nfall = 0;
  for (int64_t a = (int64_t)blockIdx.x * (kCwBlock / 32) + warp; a < N; a += nwarps) {
    uint4* const dst = reinterpret_cast<uint4*>(d + a * (int64_t)n);
    uint32_t k[32];
#pragma unroll
    for (int q = 0; q < 8; ++q) {
      const int c = lane + 32 * q;
      const uint4 v = q < 4 ? ld_stream(dst + c) : ldg_cs_if(c < nc, dst + c);
      k[4 * q] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
    }
#pragma unroll
    for (int q = 4; q < 8; ++q) {
      const bool v = lane + 32 * q < nc;
#pragma unroll
      for (int j = 0; j < 4; ++j) k[4 * q + j] = v ? k[4 * q + j] : k[0];
    }
    uint32_t umin = k[0], umax = k[0];
#pragma unroll
    for (int r = 1; r < 31; r += 2) {
      umin = __vimin3_u32(umin, k[r], k[r + 1]);
      umax = __vimax3_u32(umax, k[r], k[r + 1]);
    }
    umin = __reduce_min_sync(0xffffffffu, min(umin, k[31]));
    umax = __reduce_max_sync(0xffffffffu, max(umax, k[31]));
    const bool raw = umin > 0u && umax < 0x7F800000u;
    const uint32_t dm = __reduce_max_sync(0xffffffffu, __popc(__match_any_sync(0xffffffffu, k[0]))) >= 3 ? 3u : 0u;
    nfall += cw_sort_warp<true>(k, raw, umin, umax, dm, d + a * (int64_t)n, n, lane, cnt_sa, buf_sa, buf_ptr, one);
  }
  if (stats && lane == 0 && nfall) atomicAdd(stats, (unsigned long long)nfall);
}

}  // namespace gas


extern "C" __attribute__((visibility("default"))) int cw_info(int* regs, long long* local_bytes, int* grid_cap) {
  cudaFuncAttributes fa;
  cudaError_t e = cudaFuncSetAttribute(gas::k_fixed_cw1024, cudaFuncAttributeMaxDynamicSharedMemorySize, gas::kCwSmemBytes);
  if (e == cudaSuccess) e = cudaFuncGetAttributes(&fa, gas::k_fixed_cw1024);
  int per_sm = 0, sms = 0;
  if (e == cudaSuccess) e = cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, gas::k_fixed_cw1024, gas::kCwBlock, gas::kCwSmemBytes);
  if (e == cudaSuccess) e = cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  *regs = fa.numRegs; *local_bytes = (long long)fa.localSizeBytes; *grid_cap = per_sm * sms;
  return (int)e;
}

extern "C" __attribute__((visibility("default"))) int cw_launch(uint32_t* d, long long N, int n, unsigned long long* stats, cudaStream_t s) {
  static int cap = 0;
  if (!cap) { int r; long long l; if (cw_info(&r, &l, &cap) != 0) return -1; }
  const long long need = (N + gas::kCwBlock / 32 - 1) / (gas::kCwBlock / 32);
  const int grid = (int)(need < cap ? need : cap);
  gas::k_fixed_cw1024<<<grid, gas::kCwBlock, gas::kCwSmemBytes, s>>>(d, N, n, 1u, stats);
  return (int)cudaGetLastError();
}

// The fused default kernel (csrc/sort1024.cuh), for A/B inside the same harness.
extern "C" __attribute__((visibility("default"))) int s1_launch(uint32_t* d, long long N, int n, cudaStream_t s) {
  auto k = gas::k_fixed_sort1024<true>;
  cudaError_t e = cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, gas::kS1SmemBytes);
  int per_sm = 0, sms = 0;
  if (e == cudaSuccess) e = cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k, gas::kS1Block, gas::kS1SmemBytes);
  if (e == cudaSuccess) e = cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  if (e != cudaSuccess) return (int)e;
  const long long need = (N + gas::kS1Block / 32 - 1) / (gas::kS1Block / 32), cap = (long long)per_sm * sms;
  k<<<(int)(need < cap ? need : cap), gas::kS1Block, gas::kS1SmemBytes, s>>>(d, N, n, 1u, 0);
  return (int)cudaGetLastError();
}
