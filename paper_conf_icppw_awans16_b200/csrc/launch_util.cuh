// launch_util.cuh — host-side launch helpers shared by the kernel translation
// units of libgas.so (persistent grids sized to the
// resident blocks of all SMs, size classes).
#pragma once
#include <atomic>
#include <cstdint>
#include <cstdlib>
#include <cstring>
#include <mutex>

#include <cuda_runtime.h>

namespace gas_host {

// Host-side launch bookkeeping is cached (per device, per kernel): a call on a
// small batch is otherwise dominated by driver queries made before its first
// launch (the GPU idles meanwhile).
constexpr int kLaunchCacheDevices = 64;
inline int current_device() {
  int dev = 0;
  if (cudaGetDevice(&dev) != cudaSuccess || dev < 0 || dev >= kLaunchCacheDevices) dev = 0;
  return dev;
}
inline int num_sms() {
  static std::atomic<int> cache[kLaunchCacheDevices];  // 0 = not queried yet
  const int dev = current_device();
  int sms = cache[dev].load(std::memory_order_relaxed);
  if (sms > 0) return sms;
  if (cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev) != cudaSuccess || sms <= 0) return 148;
  cache[dev].store(sms, std::memory_order_relaxed);
  return sms;
}
// Resident blocks per SM of (kernel, threads, dynamic shared memory) on the current device, cached.
inline int occupancy_cached(const void* kernel, int threads, int smem) {
  struct Entry { const void* k; int threads, smem, dev, per_sm; };
  static std::mutex mu;
  static Entry tab[256];
  static int used = 0;
  const int dev = current_device();
  {
    std::lock_guard<std::mutex> lock(mu);
    for (int i = 0; i < used; ++i)
      if (tab[i].k == kernel && tab[i].threads == threads && tab[i].smem == smem && tab[i].dev == dev) return tab[i].per_sm;
  }
  int per_sm = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, kernel, threads, smem) != cudaSuccess || per_sm <= 0) {
    (void)cudaGetLastError();
    return 1;  // not cached: a failed query is retried next time
  }
  std::lock_guard<std::mutex> lock(mu);
  if (used < 256) tab[used++] = Entry{kernel, threads, smem, dev, per_sm};
  return per_sm;
}
// cudaFuncSetAttribute(MaxDynamicSharedMemorySize) once per (kernel, device, size).
inline cudaError_t set_smem_cached(const void* kernel, int smem) {
  struct Entry { const void* k; int smem, dev; };
  static std::mutex mu;
  static Entry tab[256];
  static int used = 0;
  const int dev = current_device();
  std::lock_guard<std::mutex> lock(mu);
  for (int i = 0; i < used; ++i)
    if (tab[i].k == kernel && tab[i].smem == smem && tab[i].dev == dev) return cudaSuccess;
  const cudaError_t e = cudaFuncSetAttribute(kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
  if (e == cudaSuccess && used < 256) tab[used++] = Entry{kernel, smem, dev};
  return e;
}

inline int32_t size_class(int64_t n) {  // smallest power of two >= n, n >= 2
  int32_t p = 2;
  while (p < n) p <<= 1;
  return p;
}

// Persistent grid: enough blocks to cover the work, at most the number of
// blocks that can be resident on all SMs at once (a multiple of the SM count).
// GAS_GRID_CAP=k (testing knob): at most k blocks per persistent launch, so that
// every block sorts many arrays back to back (tools/sanitize_cases.py).
inline int64_t grid_cap() {
  static const int64_t cap = [] {
    const char* v = std::getenv("GAS_GRID_CAP");
    return v ? (int64_t)std::atoll(v) : (int64_t)0;
  }();
  return cap;
}

template <typename K>
inline int persistent_grid(K kernel, int threads, int64_t blocks_needed) {
  const int per_sm = occupancy_cached(reinterpret_cast<const void*>(kernel), threads, 0);
  int64_t cap = (int64_t)per_sm * num_sms();
  if (grid_cap() > 0 && grid_cap() < cap) cap = grid_cap();
  return (int)(blocks_needed < cap ? (blocks_needed > 0 ? blocks_needed : 1) : cap);
}

template <typename K>
inline int persistent_grid_smem(K kernel, int threads, int smem, int64_t blocks_needed) {
  const int per_sm = occupancy_cached(reinterpret_cast<const void*>(kernel), threads, smem);
  int64_t cap = (int64_t)per_sm * num_sms();
  if (grid_cap() > 0 && grid_cap() < cap) cap = grid_cap();
  return (int)(blocks_needed < cap ? (blocks_needed > 0 ? blocks_needed : 1) : cap);
}


inline bool env_flag(const char* name) {
  const char* v = std::getenv(name);
  return v && v[0] != '\0' && std::strcmp(v, "0") != 0;
}

// Default-on switches: GAS_<NAME>=0 turns the feature off (A/B and ablations).
inline bool env_on(const char* name) {
  const char* v = std::getenv(name);
  return !(v && std::strcmp(v, "0") == 0);
}
inline bool bucket_enabled() { return env_on("GAS_BUCKET"); }       // value-bucket kernels (else networks)
inline bool sort1024_enabled() { return env_on("GAS_SORT1024"); }   // fused 1024 kernel (else bucket1024)
inline bool offsets512_bucket() { return env_on("GAS_OFFSETS512"); }  // (256, 512] offsets class on buckets

// Kernels launched by this library (gas_launch_count): one counter shared by
// every translation unit of libgas.so.
inline std::atomic<int64_t>& launch_counter() {
  static std::atomic<int64_t> c{0};
  return c;
}

// Stream-ordered device workspace from a library-owned memory pool per device
// (release threshold: keep everything, so steady-state calls allocate nothing
// from the driver and never synchronise). Captured into CUDA graphs as
// memory-allocation nodes.
inline cudaError_t ws_alloc(void** p, size_t bytes, cudaStream_t s) {
  constexpr int kMaxDev = 64;
  static std::mutex mu;
  static cudaMemPool_t pools[kMaxDev] = {};
  int dev = 0;
  cudaError_t e = cudaGetDevice(&dev);
  if (e != cudaSuccess) return e;
  if (dev < 0 || dev >= kMaxDev) return cudaErrorInvalidDevice;
  {
    std::lock_guard<std::mutex> lock(mu);
    if (!pools[dev]) {
      cudaMemPoolProps props{};
      props.allocType = cudaMemAllocationTypePinned;
      props.location.type = cudaMemLocationTypeDevice;
      props.location.id = dev;
      e = cudaMemPoolCreate(&pools[dev], &props);
      if (e != cudaSuccess) { pools[dev] = nullptr; return e; }
      uint64_t keep = ~0ull;
      cudaMemPoolSetAttribute(pools[dev], cudaMemPoolAttrReleaseThreshold, &keep);
    }
  }
  return cudaMallocFromPoolAsync(p, bytes, pools[dev], s);
}

// Host launchers, one translation unit each (built in parallel, build.py).
cudaError_t dispatch_fixed_small(bool vec, uint32_t* d, int64_t N, int n, cudaStream_t s);  // n <= 512
cudaError_t dispatch_fixed_1024(bool vec, uint32_t* d, int64_t N, int n, cudaStream_t s);   // 512 < n <= 1024
cudaError_t dispatch_fixed_cta(bool vec, uint32_t* d, int64_t N, int n, cudaStream_t s);    // 1024 < n <= 16384
cudaError_t dispatch_fixed_cluster(bool vec, uint32_t* d, int64_t N, int n, cudaStream_t s);  // 16384 < n <= 65536
// The variable-length sort (gas_api.cu; also the second pass of the two-kernel cluster path)
cudaError_t offsets_sort(uint32_t* d, const int64_t* off, int64_t N, int32_t max_len, cudaStream_t s);
cudaError_t dispatch_offsets_class(int32_t P, uint32_t* d, const int64_t* off, int64_t N, unsigned long long* ctr,
                                   cudaStream_t s);
cudaError_t dispatch_pairs(uint32_t* k, uint32_t* v, int64_t N, int n, cudaStream_t s);

}  // namespace gas_host
