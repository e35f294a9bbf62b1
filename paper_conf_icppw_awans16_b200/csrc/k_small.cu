// k_small.cu — fixed-length size classes n <= 512.
#include <cstdint>

#include <cuda_runtime.h>

#include "launch_util.cuh"
#include "segsort.cuh"
#include "bucket512.cuh"

namespace gas_host {

template <int KPT, int G, bool VEC>
cudaError_t launch_fixed_warp(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  constexpr int blk = gas::warp_block<G>();
  constexpr int smem = gas::warp_smem_bytes<KPT, G>();
  constexpr int arrays_per_block = (blk / 32) * (32 / G);
  auto k = gas::k_fixed_warp<KPT, G, VEC>;
  const cudaError_t e = set_smem_cached(reinterpret_cast<const void*>(k), smem);
  if (e != cudaSuccess) return e;
  const int grid = persistent_grid_smem(k, blk, smem, (N + arrays_per_block - 1) / arrays_per_block);
  k<<<grid, blk, smem, s>>>(d, N, n, 1u);
  return cudaGetLastError();
}



// Bucket-then-network kernel for 256 < n <= 512 with aligned rows (bucket512.cuh).
template <bool NET16>
cudaError_t launch_bucket512(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  auto k = gas::k_fixed_bucket512<NET16>;
  const cudaError_t attr = set_smem_cached(reinterpret_cast<const void*>(k), gas::kBk5SmemBytes);
  if (attr != cudaSuccess) return attr;
  const int grid = persistent_grid_smem(k, gas::kBk5Block, gas::kBk5SmemBytes, (N + GAS_BK5_WARPS - 1) / GAS_BK5_WARPS);
  k<<<grid, gas::kBk5Block, gas::kBk5SmemBytes, s>>>(d, N, n, 1u);
  return cudaGetLastError();
}

// The 16-key network branch only where most warps take it (n = 300: 5.87 ->
// 5.48 ms; it costs n = 400 / 500 about 5%, profiles/r02_ab_net16.txt).
cudaError_t launch_fixed_bucket512(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  if (GAS_BK5_NET16 && n <= gas::kBk5Net16MaxN) return launch_bucket512<true>(d, N, n, s);
  return launch_bucket512<false>(d, N, n, s);
}


// Bucket-then-network kernel for 128 < n <= 256 with aligned rows (bucket512.cuh, half a warp per array).
cudaError_t launch_fixed_bucket256(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  const cudaError_t attr = set_smem_cached(reinterpret_cast<const void*>(gas::k_fixed_bucket256), gas::kBk2SmemBytes);
  if (attr != cudaSuccess) return attr;
  const int grid = persistent_grid_smem(gas::k_fixed_bucket256, gas::kBk2Block, gas::kBk2SmemBytes,
                                        (N + 2 * GAS_BK2_WARPS - 1) / (2 * GAS_BK2_WARPS));
  gas::k_fixed_bucket256<<<grid, gas::kBk2Block, gas::kBk2SmemBytes, s>>>(d, N, n, 1u);
  return cudaGetLastError();
}

template <bool VEC>
cudaError_t dispatch_small(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  switch (size_class(n)) {
    case 2: return launch_fixed_warp<2, 1, false>(d, N, n, s);
    case 4: return launch_fixed_warp<4, 1, VEC>(d, N, n, s);
    case 8: return launch_fixed_warp<8, 1, VEC>(d, N, n, s);
    case 16: return launch_fixed_warp<16, 1, VEC>(d, N, n, s);
    case 32: return launch_fixed_warp<32, 1, VEC>(d, N, n, s);
    case 64: return launch_fixed_warp<32, 2, VEC>(d, N, n, s);
    case 128: return launch_fixed_warp<32, 4, VEC>(d, N, n, s);
    case 256:
      if (VEC && bucket_enabled() && n > 128) return launch_fixed_bucket256(d, N, n, s);
      return launch_fixed_warp<32, 8, VEC>(d, N, n, s);
    case 512:
      if (VEC && bucket_enabled()) return launch_fixed_bucket512(d, N, n, s);
      return launch_fixed_warp<32, 16, VEC>(d, N, n, s);
  }
  return cudaErrorInvalidValue;
}

cudaError_t dispatch_fixed_small(bool vec, uint32_t* d, int64_t N, int n, cudaStream_t s) {
  return vec ? dispatch_small<true>(d, N, n, s) : dispatch_small<false>(d, N, n, s);
}

}  // namespace gas_host
