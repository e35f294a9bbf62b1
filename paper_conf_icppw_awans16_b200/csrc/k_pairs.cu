// k_pairs.cu — the stable key + payload variant.
#include <cstdint>

#include <cuda_runtime.h>

#include "launch_util.cuh"
#include "pairs.cuh"
#include "pairs1024.cuh"

namespace gas_host {

template <int KPT, int G, int W>
cudaError_t launch_pairs(uint32_t* k, uint32_t* v, int64_t N, int n, cudaStream_t s, const uint32_t* list = nullptr) {
  using C = gas::PairsCfg<KPT, G, W>;
  auto kern = gas::k_pairs<KPT, G, W>;
  cudaError_t e = set_smem_cached(reinterpret_cast<const void*>(kern), C::SMEM);
  if (e != cudaSuccess) return e;
  int per_sm = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, kern, C::TPB, C::SMEM) != cudaSuccess || per_sm <= 0)
    per_sm = 1;
  const int64_t need = (N + C::GROUPS - 1) / C::GROUPS;
  const int64_t cap = (int64_t)per_sm * num_sms();
  kern<<<(int)(need < cap ? need : cap), C::TPB, C::SMEM, s>>>(k, v, N, n, list);
  return cudaGetLastError();
}

// 512 < n <= 1024, 16-byte-aligned key and payload rows: the bucket kernel
// (pairs1024.cuh), then the network kernel over the arrays it listed.
// GAS_PAIRS_BUCKET=0: the network kernel for every array (A/B).
cudaError_t launch_pairs_bucket1024(uint32_t* k, uint32_t* v, int64_t N, int n, cudaStream_t s) {
  void* ws = nullptr;
  cudaError_t e = ws_alloc(&ws, 4 * ((size_t)N + 1), s);
  if (e != cudaSuccess) return e;
  uint32_t* fail = static_cast<uint32_t*>(ws);
  e = cudaMemsetAsync(fail, 0, 4, s);
  if (e == cudaSuccess)
    e = set_smem_cached(reinterpret_cast<const void*>(gas::k_pairs_bucket1024), gas::kPbSmemBytes);
  if (e == cudaSuccess) {
    const int grid = persistent_grid_smem(gas::k_pairs_bucket1024, gas::kPbBlock, gas::kPbSmemBytes,
                                          (N + gas::kPbBlock / 32 - 1) / (gas::kPbBlock / 32));
    gas::k_pairs_bucket1024<<<grid, gas::kPbBlock, gas::kPbSmemBytes, s>>>(k, v, N, n, fail);
    e = cudaGetLastError();
  }
  if (e == cudaSuccess) e = launch_pairs<32, 32, 1>(k, v, N, n, s, fail);
  const cudaError_t f = cudaFreeAsync(ws, s);
  if (e == cudaSuccess) launch_counter() += 1;  // the caller counts one launch
  return e != cudaSuccess ? e : f;
}

cudaError_t dispatch_pairs(uint32_t* k, uint32_t* v, int64_t N, int n, cudaStream_t s) {
  const bool aligned = n % 4 == 0 && (reinterpret_cast<uintptr_t>(k) & 15u) == 0 &&
                       (reinterpret_cast<uintptr_t>(v) & 15u) == 0;
  if (n > 512 && n <= 1024 && aligned && N < (int64_t(1) << 32) && env_on("GAS_PAIRS_BUCKET"))
    return launch_pairs_bucket1024(k, v, N, n, s);
  switch (size_class(n)) {
    case 2: return launch_pairs<2, 1, 1>(k, v, N, n, s);
    case 4: return launch_pairs<4, 1, 1>(k, v, N, n, s);
    case 8: return launch_pairs<8, 1, 1>(k, v, N, n, s);
    case 16: return launch_pairs<16, 1, 1>(k, v, N, n, s);
    case 32: return launch_pairs<32, 1, 1>(k, v, N, n, s);
    case 64: return launch_pairs<32, 2, 1>(k, v, N, n, s);
    case 128: return launch_pairs<32, 4, 1>(k, v, N, n, s);
    case 256: return launch_pairs<32, 8, 1>(k, v, N, n, s);
    case 512: return launch_pairs<32, 16, 1>(k, v, N, n, s);
    case 1024: return launch_pairs<32, 32, 1>(k, v, N, n, s);
    case 2048: return launch_pairs<32, 32, 2>(k, v, N, n, s);
    case 4096: return launch_pairs<32, 32, 4>(k, v, N, n, s);
    case 8192: return launch_pairs<32, 32, 8>(k, v, N, n, s);
  }
  return cudaErrorInvalidValue;
}

}  // namespace gas_host
