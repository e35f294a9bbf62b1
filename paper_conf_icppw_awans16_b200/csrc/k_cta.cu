// k_cta.cu — fixed-length classes 1024 < n <= 16384, one CTA (group) per array.
#include <cstdint>

#include <cuda_runtime.h>

#include "launch_util.cuh"
#include "segsort.cuh"
#include "bucket_cta.cuh"

namespace gas_host {

template <int W, int WR, bool VEC>
cudaError_t launch_fixed_cta(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  auto k = gas::k_fixed_cta<W, WR, VEC>;
  constexpr int smem = gas::cta_smem_bytes<W, WR>();
  const cudaError_t e = set_smem_cached(reinterpret_cast<const void*>(k), smem);
  if (e != cudaSuccess) return e;
  k<<<persistent_grid_smem(k, 32 * WR, smem, N), 32 * WR, smem, s>>>(d, N, n, 1u);
  return cudaGetLastError();
}


// Bucket-then-network, one array per CTA of W warps (bucket_cta.cuh).
template <int W, int WR, bool VEC>
cudaError_t launch_fixed_bucket_cta(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  auto k = gas::k_fixed_bucket_cta<W, WR, VEC>;
  constexpr int gr = gas::bkc_groups<WR>(), blk = gas::bkc_block<WR>();
  constexpr int smem = gas::BkCta<W, WR>::SMEM * gr;
  const cudaError_t e = set_smem_cached(reinterpret_cast<const void*>(k), smem);
  if (e != cudaSuccess) return e;
  k<<<persistent_grid_smem(k, blk, smem, (N + gr - 1) / gr), blk, smem, s>>>(d, N, n, 1u);
  return cudaGetLastError();
}


// Fixed-length CTA classes (n > 1024): W warps' network, WR = ceil(n / 1024) real
// warps rounded to the instantiated set (padding blocks are virtual, see sort_cta).
template <bool VEC>
cudaError_t dispatch_cta(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  if (bucket_enabled()) {
    if (n <= 2048) return launch_fixed_bucket_cta<2, 2, VEC>(d, N, n, s);
    if (n <= 3072) return launch_fixed_bucket_cta<4, 3, VEC>(d, N, n, s);
    if (n <= 4096) return launch_fixed_bucket_cta<4, 4, VEC>(d, N, n, s);
    if (n <= 6144) return launch_fixed_bucket_cta<8, 6, VEC>(d, N, n, s);
    if (n <= 8192) return launch_fixed_bucket_cta<8, 8, VEC>(d, N, n, s);
    if (n <= 12288) return launch_fixed_bucket_cta<16, 12, VEC>(d, N, n, s);
    return launch_fixed_bucket_cta<16, 16, VEC>(d, N, n, s);
  }
  if (n <= 2048) return launch_fixed_cta<2, 2, VEC>(d, N, n, s);
  if (n <= 3072) return launch_fixed_cta<4, 3, VEC>(d, N, n, s);
  if (n <= 4096) return launch_fixed_cta<4, 4, VEC>(d, N, n, s);
  if (n <= 6144) return launch_fixed_cta<8, 6, VEC>(d, N, n, s);
  if (n <= 8192) return launch_fixed_cta<8, 8, VEC>(d, N, n, s);
  if (n <= 12288) return launch_fixed_cta<16, 12, VEC>(d, N, n, s);
  return launch_fixed_cta<16, 16, VEC>(d, N, n, s);
}


cudaError_t dispatch_fixed_cta(bool vec, uint32_t* d, int64_t N, int n, cudaStream_t s) {
  return vec ? dispatch_cta<true>(d, N, n, s) : dispatch_cta<false>(d, N, n, s);
}

}  // namespace gas_host
