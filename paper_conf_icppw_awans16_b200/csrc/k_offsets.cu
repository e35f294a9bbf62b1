// k_offsets.cu — the variable-length (CSR offsets) size classes.
#include <cstdint>

#include <cuda_runtime.h>

#include "launch_util.cuh"
#include "segsort.cuh"
#include "bucket_cta.cuh"

namespace gas_host {

template <int W, int WR, int RV = 16>
cudaError_t launch_offsets_bucket(uint32_t* d, const int64_t* off, int64_t N, int64_t lo, int64_t hi,
                                  unsigned long long* ctr, cudaStream_t s) {
  auto k = gas::k_offsets_bucket<W, WR, RV>;
  constexpr int gr = 1, blk = 32 * WR;
  constexpr int smem = gas::BkCta<W, WR>::SMEM * gr;
  const cudaError_t e = set_smem_cached(reinterpret_cast<const void*>(k), smem);
  if (e != cudaSuccess) return e;
  k<<<persistent_grid_smem(k, blk, smem, ((N + 31) / 32 + gr - 1) / gr), blk, smem, s>>>(d, off, N, lo, hi, ctr, 1u);
  return cudaGetLastError();
}


template <int KPT, int G>
cudaError_t launch_offsets_warp(uint32_t* d, const int64_t* off, int64_t N, cudaStream_t s) {
  constexpr int blk = gas::warp_block<G>();
  constexpr int smem = gas::warp_smem_bytes<KPT, G>();
  auto k = gas::k_offsets_warp<KPT, G>;
  const cudaError_t e = set_smem_cached(reinterpret_cast<const void*>(k), smem);
  if (e != cudaSuccess) return e;
  const int64_t windows = (N + 31) / 32;
  const int grid = persistent_grid_smem(k, blk, smem, (windows + blk / 32 - 1) / (blk / 32));
  k<<<grid, blk, smem, s>>>(d, off, N, 1u);
  return cudaGetLastError();
}

template <int W, int WR>
cudaError_t launch_offsets_cta(uint32_t* d, const int64_t* off, int64_t N, int64_t lo, int64_t hi,
                               unsigned long long* ctr, cudaStream_t s) {
  auto k = gas::k_offsets_cta<W, WR>;
  constexpr int smem = gas::cta_smem_bytes<W, WR>();
  const cudaError_t e = set_smem_cached(reinterpret_cast<const void*>(k), smem);
  if (e != cudaSuccess) return e;
  k<<<persistent_grid_smem(k, 32 * WR, smem, (N + 31) / 32), 32 * WR, smem, s>>>(d, off, N, lo, hi, ctr, 1u);
  return cudaGetLastError();
}

cudaError_t dispatch_offsets_class(int32_t P, uint32_t* d, const int64_t* off, int64_t N, unsigned long long* ctr,
                                   cudaStream_t s) {
  switch (P) {
    case 2: return launch_offsets_warp<2, 1>(d, off, N, s);
    case 4: return launch_offsets_warp<4, 1>(d, off, N, s);
    case 8: return launch_offsets_warp<8, 1>(d, off, N, s);
    case 16: return launch_offsets_warp<16, 1>(d, off, N, s);
    case 32: return launch_offsets_warp<32, 1>(d, off, N, s);
    case 64: return launch_offsets_warp<32, 2>(d, off, N, s);
    case 128: return launch_offsets_warp<32, 4>(d, off, N, s);
    case 256: return launch_offsets_warp<32, 8>(d, off, N, s);
    case 512:
      if (bucket_enabled() && offsets512_bucket()) return launch_offsets_bucket<1, 1, 8>(d, off, N, 256, 512, ctr + 8, s);
      return launch_offsets_warp<32, 16>(d, off, N, s);
    case 1024:
      if (bucket_enabled()) return launch_offsets_bucket<1, 1>(d, off, N, 512, 1024, ctr + 7, s);
      return launch_offsets_warp<32, 32>(d, off, N, s);
    case 2048:
      if (bucket_enabled()) return launch_offsets_bucket<2, 2>(d, off, N, 1024, 2048, ctr, s);
      return launch_offsets_cta<2, 2>(d, off, N, 1024, 2048, ctr, s);
    case 3072:
      if (bucket_enabled()) return launch_offsets_bucket<4, 3>(d, off, N, 2048, 3072, ctr + 1, s);
      return launch_offsets_cta<4, 3>(d, off, N, 2048, 3072, ctr + 1, s);
    case 4096:
      if (bucket_enabled()) return launch_offsets_bucket<4, 4>(d, off, N, 3072, 4096, ctr + 2, s);
      return launch_offsets_cta<4, 4>(d, off, N, 3072, 4096, ctr + 2, s);
    case 6144:
      if (bucket_enabled()) return launch_offsets_bucket<8, 6>(d, off, N, 4096, 6144, ctr + 3, s);
      return launch_offsets_cta<8, 6>(d, off, N, 4096, 6144, ctr + 3, s);
    case 8192:
      if (bucket_enabled()) return launch_offsets_bucket<8, 8>(d, off, N, 6144, 8192, ctr + 4, s);
      return launch_offsets_cta<8, 8>(d, off, N, 6144, 8192, ctr + 4, s);
    case 12288:
      if (bucket_enabled()) return launch_offsets_bucket<16, 12>(d, off, N, 8192, 12288, ctr + 5, s);
      return launch_offsets_cta<16, 12>(d, off, N, 8192, 12288, ctr + 5, s);
    case 16384:
      if (bucket_enabled()) return launch_offsets_bucket<16, 16>(d, off, N, 12288, 16384, ctr + 6, s);
      return launch_offsets_cta<16, 16>(d, off, N, 12288, 16384, ctr + 6, s);
  }
  return cudaErrorInvalidValue;
}

}  // namespace gas_host
