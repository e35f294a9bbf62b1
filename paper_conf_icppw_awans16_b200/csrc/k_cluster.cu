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
template <int W, int WR, int C, int MAXN, bool PART = false>
cudaError_t launch_cluster(uint32_t* d, int64_t N, int n, uint32_t* fail, int64_t* parts, cudaStream_t s) {
  using G = gas::ClCfg<W, WR, C, MAXN>;
  auto k = gas::k_cluster_sort<W, WR, C, MAXN, PART>;
  constexpr int smem = PART ? 0 : G::SMEM;
  cudaError_t e = set_smem_cached(reinterpret_cast<const void*>(k), smem);
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
  cfg.dynamicSmemBytes = smem;
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
  return cudaLaunchKernelEx(&cfg, k, d, N, n, 1u, fail, parts);
}

// Two-kernel path (n > 32768): the cluster kernel only partitions each array
// into 8 value-range parts in place and writes their boundaries as a CSR of
// 8 N parts; the variable-length sort (offsets_sort, the CTA bucket classes)
// then sorts every part. Each array crosses HBM twice (16 n bytes), but both
// kernels keep every SM busy, where the one-kernel path (n <= 32768) walks
// each cluster's arrays through five dependent phases.
cudaError_t dispatch_fixed_cluster(bool vec, uint32_t* d, int64_t N, int n, cudaStream_t s) {
  (void)vec;  // rows at any 4-byte alignment: scalar part sorts
  // measured (profiles/r02_sweep_f4.txt): one pass 0.11-0.12 of HBM for n <= 32768, 0.07 above;
  // two kernels 0.07-0.10 for n <= 32768, 0.107-0.112 above
  const char* ov = std::getenv("GAS_CLUSTER_ONEPASS");  // tests / A/B: 1 one pass, 0 two kernels
  const bool onepass = ov && ov[0] ? std::atoi(ov) != 0 : n <= 32768;
  void* ws = nullptr;
  const size_t fail_bytes = (4 * ((size_t)N + 1) + 7) & ~(size_t)7;
  cudaError_t e = ws_alloc(&ws, fail_bytes + (onepass ? 0 : 8 * ((size_t)N * 8 + 1)), s);
  if (e != cudaSuccess) return e;
  uint32_t* fail = static_cast<uint32_t*>(ws);
  int64_t* parts = onepass ? nullptr : reinterpret_cast<int64_t*>(static_cast<unsigned char*>(ws) + fail_bytes);
  e = cudaMemsetAsync(fail, 0, 4, s);
  if (e == cudaSuccess) {
    if (!onepass) {
      e = launch_cluster<8, 8, 8, 65536, true>(d, N, n, fail, parts, s);  // 256-thread CTAs, no dynamic shared memory
      if (e == cudaSuccess) {
        launch_counter() += 1;
        e = offsets_sort(d, parts, N * 8, gas::kClPartMaxOff, s);  // counts its own launches
      }
    } else {
      // CTAs sized to their part (cluster_sort.cuh): parts of ~2-4 K keys
      if (n <= 24576) e = launch_cluster<4, 4, 8, 24576>(d, N, n, fail, nullptr, s);
      else if (n <= 32768) e = launch_cluster<8, 5, 8, 32768>(d, N, n, fail, nullptr, s);
      else e = launch_cluster<16, 12, 8, 65536>(d, N, n, fail, nullptr, s);  // (16-CTA clusters of <4,4> / <8,5>: 2-4x slower)
      if (e == cudaSuccess) launch_counter() += 1;
    }
  }
  if (e == cudaSuccess) {
    gas::k_cluster_fallback<<<num_sms(), 1024, 0, s>>>(d, n, fail);
    e = cudaGetLastError();
  }
  const cudaError_t f = cudaFreeAsync(ws, s);
  if (e == cudaSuccess) launch_counter() += 1;
  return e != cudaSuccess ? e : f;
}

}  // namespace gas_host
