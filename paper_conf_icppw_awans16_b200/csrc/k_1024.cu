// k_1024.cu — the 512 < n <= 1024 class (configs[1]'s n = 1000): fused bucket /
// counting-sort kernel (sort1024.cuh), plus the earlier kernels for A/B.
#include <cstdint>

#include <cuda_runtime.h>

#include "launch_util.cuh"
#include "segsort.cuh"
#include "bucket1024.cuh"
#include "sort1024.cuh"
#include "split1024.cuh"

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



cudaError_t launch_fixed_1024_tma(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  // per-device attribute: set on every call (cheap), the current device may change
  const cudaError_t attr = set_smem_cached(reinterpret_cast<const void*>(gas::k_fixed_1024_tma), gas::kTmaSmemBytes);
  if (attr != cudaSuccess) return attr;
  int per_sm = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, gas::k_fixed_1024_tma, gas::kWarpBlock,
                                                    gas::kTmaSmemBytes) != cudaSuccess || per_sm <= 0)
    per_sm = 1;
  const int64_t need = (N + gas::kWarpBlock / 32 - 1) / (gas::kWarpBlock / 32);
  const int64_t cap = (int64_t)per_sm * num_sms();
  const int grid = (int)(need < cap ? need : cap);
  gas::k_fixed_1024_tma<<<grid, gas::kWarpBlock, gas::kTmaSmemBytes, s>>>(d, N, n, 1u);
  return cudaGetLastError();
}

// Bucket-then-network kernel for 512 < n <= 1024 with aligned rows
// (bucket1024.cuh). Default on; GAS_BUCKET=0 selects the pure network.
template <bool VEC>
cudaError_t launch_fixed_bucket1024(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  auto k = VEC ? gas::k_fixed_bucket1024<false> : gas::k_fixed_bucket1024_any<false, false>;
  const cudaError_t attr = set_smem_cached(reinterpret_cast<const void*>(k), gas::kBkSmemBytes);
  if (attr != cudaSuccess) return attr;
  const int grid = persistent_grid_smem(k, gas::kBkBlock, gas::kBkSmemBytes,
                                        (N + gas::kBkBlock / 32 - 1) / (gas::kBkBlock / 32));
  k<<<grid, gas::kBkBlock, gas::kBkSmemBytes, s>>>(d, N, n, 1u, nullptr);
  return cudaGetLastError();
}

// Default for 512 < n <= 1024: value buckets, counting sort where they do not
// fit, network as the last resort (sort1024.cuh). GAS_SORT1024=0 selects the
// previous bucket-then-network kernel (A/B).
template <bool VEC>
cudaError_t launch_fixed_sort1024(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  auto k = gas::k_fixed_sort1024<VEC>;
  const cudaError_t attr = set_smem_cached(reinterpret_cast<const void*>(k), gas::kS1SmemBytes);
  if (attr != cudaSuccess) return attr;
  const int grid = persistent_grid_smem(k, gas::kS1Block, gas::kS1SmemBytes,
                                        (N + gas::kS1Block / 32 - 1) / (gas::kS1Block / 32));
  const char* mv = std::getenv("GAS_SORT1024_MODE");  // tests / ablations: 0 auto, 1 counting sort, 2 network, 3 no predictor
  const int mode = mv ? std::atoi(mv) : 0;
  k<<<grid, gas::kS1Block, gas::kS1SmemBytes, s>>>(d, N, n, 1u, mode);
  return cudaGetLastError();
}


// Default for large batches: the device-routed pipeline of sort1024.cuh
// (sampler -> bucket kernel -> key-linear and batch-CDF bucket kernels (16-byte rows) -> counting-sort kernel -> split kernel), 6 (4)
// launches and 4 N + 8 bytes of stream-ordered workspace.
template <bool VEC>
cudaError_t launch_s1_pipeline(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  void* ws = nullptr;
  cudaError_t e = ws_alloc(&ws, sizeof(gas::S1Ctl) + 4 * (size_t)N, s);
  if (e != cudaSuccess) return e;
  gas::S1Ctl* ctl = static_cast<gas::S1Ctl*>(ws);
  const char* fv = std::getenv("GAS_S1_FORCE");  // tests / ablations: 0 bucket, 1 counting sort, 2 split kernel, 3 key-linear buckets, 4 batch-CDF buckets
  const uint32_t force = fv && fv[0] ? (uint32_t)std::atoi(fv) : 0xFFFFFFFFu;
  gas::k_s1_sample<VEC><<<1, 1024, 0, s>>>(d, N, n, ctl, force);
  e = cudaGetLastError();
  if (e == cudaSuccess) {
    auto k = VEC ? gas::k_fixed_bucket1024<true> : gas::k_fixed_bucket1024_any<false, true>;
    e = set_smem_cached(reinterpret_cast<const void*>(k), gas::kBkSmemBytes);
    if (e == cudaSuccess) {
      const int grid = persistent_grid_smem(k, gas::kBkBlock, gas::kBkSmemBytes,
                                            (N + gas::kBkBlock / 32 - 1) / (gas::kBkBlock / 32));
      k<<<grid, gas::kBkBlock, gas::kBkSmemBytes, s>>>(d, N, n, 1u, ctl);
      e = cudaGetLastError();
    }
  }
  // key-linear and batch-CDF bucket kernels (16-byte rows only)
  for (int map = gas::kMapKeyLin; VEC && map <= gas::kMapCdf && e == cudaSuccess; ++map) {
    auto k = map == gas::kMapKeyLin ? gas::k_fixed_bucket1024<true, gas::kMapKeyLin>
                                    : gas::k_fixed_bucket1024<true, gas::kMapCdf>;
    const int smem = gas::kBkSmemBytes + (map == gas::kMapCdf ? gas::kCdfEntries * 8 : 0);
    e = set_smem_cached(reinterpret_cast<const void*>(k), smem);
    if (e == cudaSuccess) {
      const int grid = persistent_grid_smem(k, gas::kBkBlock, smem, (N + gas::kBkBlock / 32 - 1) / (gas::kBkBlock / 32));
      k<<<grid, gas::kBkBlock, smem, s>>>(d, N, n, 1u, ctl);
      e = cudaGetLastError();
    }
  }
  if (e == cudaSuccess) {
    auto k = gas::k_s1_count<VEC>;
    e = set_smem_cached(reinterpret_cast<const void*>(k), gas::kCwSmemBytes);
    if (e == cudaSuccess) {
      const int grid = persistent_grid_smem(k, gas::kCwBlock, gas::kCwSmemBytes,
                                            (N + gas::kCwBlock / 32 - 1) / (gas::kCwBlock / 32));
      k<<<grid, gas::kCwBlock, gas::kCwSmemBytes, s>>>(d, N, n, 1u, ctl);
      e = cudaGetLastError();
    }
  }
  if (e == cudaSuccess) {
    auto k = gas::k_s1_split<VEC>;
    e = set_smem_cached(reinterpret_cast<const void*>(k), gas::kSpSmemBytes);
    if (e == cudaSuccess) {
      const int grid = persistent_grid_smem(k, gas::kSpBlock, gas::kSpSmemBytes,
                                            (N + gas::kSpBlock / 32 - 1) / (gas::kSpBlock / 32));
      k<<<grid, gas::kSpBlock, gas::kSpSmemBytes, s>>>(d, N, n, 1u, ctl);
      e = cudaGetLastError();
    }
  }
  const cudaError_t f = cudaFreeAsync(ws, s);  // stream-ordered: after the kernels
  if (e == cudaSuccess) launch_counter() += VEC ? 6 : 4;
  return e != cudaSuccess ? e : f;
}

// Batches of at least this many arrays take the pipeline; smaller ones the
// single fused kernel (one launch, no workspace: latency of serving-size batches).
inline int64_t s1_pipeline_min() {
  const char* v = std::getenv("GAS_S1_PIPELINE_MIN");
  return v ? std::atoll(v) : 16384;
}

template <bool VEC>
cudaError_t dispatch_1024(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  // TMA-prefetch variant: opt-in (GAS_TMA=1). Measured on B200 it removes the
  // global-load stalls but is 5% slower overall (profiles/r01_ab_tma.txt).
  if (VEC && env_flag("GAS_TMA")) {
    launch_counter() += 1;
    return launch_fixed_1024_tma(d, N, n, s);
  }
  if (bucket_enabled() && sort1024_enabled()) {
    const char* mv = std::getenv("GAS_SORT1024_MODE");  // a forced branch runs in the fused kernel
    if ((!mv || std::atoi(mv) == 0) && N >= s1_pipeline_min() && N < (int64_t(1) << 32))
      return launch_s1_pipeline<VEC>(d, N, n, s);  // counts its own 6 (4) launches
    launch_counter() += 1;
    return launch_fixed_sort1024<VEC>(d, N, n, s);
  }
  launch_counter() += 1;
  if (bucket_enabled()) return launch_fixed_bucket1024<VEC>(d, N, n, s);
  return launch_fixed_warp<32, 32, VEC>(d, N, n, s);
}

cudaError_t dispatch_fixed_1024(bool vec, uint32_t* d, int64_t N, int n, cudaStream_t s) {
  return vec ? dispatch_1024<true>(d, N, n, s) : dispatch_1024<false>(d, N, n, s);
}

}  // namespace gas_host
