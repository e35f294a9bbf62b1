// k_pairs.cu — the stable key + payload variant.
#include <cstdint>

#include <cuda_runtime.h>

#include "launch_util.cuh"
#include "pairs.cuh"

namespace gas_host {

template <int KPT, int G, int W>
cudaError_t launch_pairs(uint32_t* k, uint32_t* v, int64_t N, int n, cudaStream_t s) {
  using C = gas::PairsCfg<KPT, G, W>;
  auto kern = gas::k_pairs<KPT, G, W>;
  cudaError_t e = cudaFuncSetAttribute(kern, cudaFuncAttributeMaxDynamicSharedMemorySize, C::SMEM);
  if (e != cudaSuccess) return e;
  int per_sm = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, kern, C::TPB, C::SMEM) != cudaSuccess || per_sm <= 0)
    per_sm = 1;
  const int64_t need = (N + C::GROUPS - 1) / C::GROUPS;
  const int64_t cap = (int64_t)per_sm * num_sms();
  kern<<<(int)(need < cap ? need : cap), C::TPB, C::SMEM, s>>>(k, v, N, n);
  return cudaGetLastError();
}

cudaError_t dispatch_pairs(uint32_t* k, uint32_t* v, int64_t N, int n, cudaStream_t s) {
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
