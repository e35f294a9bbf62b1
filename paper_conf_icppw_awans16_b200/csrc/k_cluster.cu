// k_cluster.cu — fixed-length arrays of 16384 < n <= 65536 (SURVEY.md §8(f)
// row f4): one 8-CTA thread-block cluster per array (cluster_sort.cuh), then
// the fallback kernel for the rare arrays with an oversize part.
#include <cstdint>

#include <cuda_runtime.h>

#include "launch_util.cuh"
#include "segsort.cuh"
#include "cluster_sort.cuh"

namespace gas_host {

cudaError_t dispatch_fixed_cluster(bool vec, uint32_t* d, int64_t N, int n, cudaStream_t s) {
  (void)vec;  // rows at any 4-byte alignment: scalar part sorts
  void* ws = nullptr;
  cudaError_t e = ws_alloc(&ws, 4 * ((size_t)N + 1), s);
  if (e != cudaSuccess) return e;
  uint32_t* fail = static_cast<uint32_t*>(ws);
  e = cudaMemsetAsync(fail, 0, 4, s);
  if (e == cudaSuccess) e = cudaFuncSetAttribute(gas::k_cluster_sort, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                                 gas::kClSmem);
  if (e == cudaSuccess) {
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3(gas::kClC, 1, 1);
    cfg.blockDim = dim3(gas::kClT, 1, 1);
    cfg.dynamicSmemBytes = gas::kClSmem;
    cfg.stream = s;
    int clusters = 0;
    if (cudaOccupancyMaxActiveClusters(&clusters, gas::k_cluster_sort, &cfg) != cudaSuccess || clusters <= 0)
      clusters = num_sms() / gas::kClC;
    if (clusters < 1) clusters = 1;
    const int64_t need = N < clusters ? N : clusters;
    gas::k_cluster_sort<<<(unsigned)(need * gas::kClC), gas::kClT, gas::kClSmem, s>>>(d, N, n, 1u, fail);
    e = cudaGetLastError();
  }
  if (e == cudaSuccess) {
    gas::k_cluster_fallback<<<num_sms(), 1024, 0, s>>>(d, n, fail);
    e = cudaGetLastError();
  }
  const cudaError_t f = cudaFreeAsync(ws, s);
  if (e == cudaSuccess) launch_counter() += 2;
  return e != cudaSuccess ? e : f;
}

}  // namespace gas_host
