// k_cluster.cu — fixed-length arrays of 16384 < n <= 65536 (SURVEY.md §8(f)
// row f4): one thread-block cluster of 8 or 16 CTAs per array
// (cluster_sort.cuh), then the fallback kernel for the rare arrays with an
// oversize part.
#include <cstdint>

#include <cuda_runtime.h>

#include "launch_util.cuh"
#include "segsort.cuh"
#include "cluster_sort.cuh"

namespace gas_host {

// Persistent launch of k_cluster_sort<W, WR, C, MAXN>: as many clusters as fit
// at once (cudaOccupancyMaxActiveClusters), each looping over arrays.
template <int W, int WR, int C, int MAXN>
cudaError_t launch_cluster(uint32_t* d, int64_t N, int n, uint32_t* fail, cudaStream_t s) {
  using G = gas::ClCfg<W, WR, C, MAXN>;
  auto k = gas::k_cluster_sort<W, WR, C, MAXN>;
  cudaError_t e = cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, G::SMEM);
  if (e == cudaSuccess && C > 8) e = cudaFuncSetAttribute(k, cudaFuncAttributeNonPortableClusterSizeAllowed, 1);
  if (e != cudaSuccess) return e;
  cudaLaunchAttribute attr[1];
  attr[0].id = cudaLaunchAttributeClusterDimension;
  attr[0].val.clusterDim.x = C;
  attr[0].val.clusterDim.y = 1;
  attr[0].val.clusterDim.z = 1;
  cudaLaunchConfig_t cfg = {};
  cfg.gridDim = dim3(C, 1, 1);
  cfg.blockDim = dim3(G::T, 1, 1);
  cfg.dynamicSmemBytes = G::SMEM;
  cfg.stream = s;
  cfg.attrs = attr;
  cfg.numAttrs = 1;
  int clusters = 0;
  if (cudaOccupancyMaxActiveClusters(&clusters, k, &cfg) != cudaSuccess || clusters <= 0) {
    (void)cudaGetLastError();  // clear a failed query
    clusters = num_sms() / C;
  }
  if (clusters < 1) clusters = 1;
  const int64_t need = N < clusters ? N : clusters;
  cfg.gridDim = dim3((unsigned)(need * C), 1, 1);
  return cudaLaunchKernelEx(&cfg, k, d, N, n, 1u, fail);
}

cudaError_t dispatch_fixed_cluster(bool vec, uint32_t* d, int64_t N, int n, cudaStream_t s) {
  (void)vec;  // rows at any 4-byte alignment: scalar part sorts
  void* ws = nullptr;
  cudaError_t e = ws_alloc(&ws, 4 * ((size_t)N + 1), s);
  if (e != cudaSuccess) return e;
  uint32_t* fail = static_cast<uint32_t*>(ws);
  e = cudaMemsetAsync(fail, 0, 4, s);
  if (e == cudaSuccess) {
    // CTAs sized to their part (cluster_sort.cuh): parts of ~2-4 K keys
    if (n <= 24576) e = launch_cluster<4, 4, 8, 24576>(d, N, n, fail, s);
    else if (n <= 32768) e = launch_cluster<8, 5, 8, 32768>(d, N, n, fail, s);
    else e = launch_cluster<16, 12, 8, 65536>(d, N, n, fail, s);  // (16-CTA clusters of <4,4> / <8,5>: 2-4x slower)
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
