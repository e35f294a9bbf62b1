// gas_api.cu — the C ABI of include/gas.h: argument validation, size-class
// dispatch, launch configuration and status codes.
#include <atomic>
#include <map>
#include <mutex>
#include <cstdint>
#include <cstdlib>
#include <cstring>

#include <cuda_runtime.h>

#include "../../include/gas.h"
#include "segsort.cuh"
#include "bucket1024.cuh"
#include "bucket512.cuh"
#include "bucket_cta.cuh"
#include "pairs.cuh"

namespace {

constexpr int32_t kMaxPairsLen = 8192;  // 64-bit network elements: 8 KB of SMEM per 1024
constexpr int32_t kMaxLen = 16384;  // 4x the spectra bound of P:L170-173

thread_local int g_last_cuda_error = 0;
std::atomic<int64_t> g_launches{0};

gas_status cuda_fail(cudaError_t e) {
  g_last_cuda_error = (int)e;
  return GAS_ERROR_CUDA;
}

int num_sms() {
  int dev = 0, sms = 0;
  if (cudaGetDevice(&dev) != cudaSuccess) return 148;
  if (cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev) != cudaSuccess || sms <= 0) return 148;
  return sms;
}

int32_t size_class(int64_t n) {  // smallest power of two >= n, n >= 2
  int32_t p = 2;
  while (p < n) p <<= 1;
  return p;
}

// Persistent grid: enough blocks to cover the work, at most the number of
// blocks that can be resident on all SMs at once (a multiple of the SM count).
// GAS_GRID_CAP=k (testing knob): at most k blocks per persistent launch, so that
// every block sorts many arrays back to back (tools/sanitize_cases.py).
int64_t grid_cap() {
  static const int64_t cap = [] {
    const char* v = std::getenv("GAS_GRID_CAP");
    return v ? (int64_t)std::atoll(v) : (int64_t)0;
  }();
  return cap;
}

template <typename K>
int persistent_grid(K kernel, int threads, int64_t blocks_needed) {
  int per_sm = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, kernel, threads, 0) != cudaSuccess || per_sm <= 0)
    per_sm = 1;
  int64_t cap = (int64_t)per_sm * num_sms();
  if (grid_cap() > 0 && grid_cap() < cap) cap = grid_cap();
  return (int)(blocks_needed < cap ? (blocks_needed > 0 ? blocks_needed : 1) : cap);
}

template <typename K>
int persistent_grid_smem(K kernel, int threads, int smem, int64_t blocks_needed) {
  int per_sm = 0;
  if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, kernel, threads, smem) != cudaSuccess || per_sm <= 0)
    per_sm = 1;
  int64_t cap = (int64_t)per_sm * num_sms();
  if (grid_cap() > 0 && grid_cap() < cap) cap = grid_cap();
  return (int)(blocks_needed < cap ? (blocks_needed > 0 ? blocks_needed : 1) : cap);
}

template <int KPT, int G, bool VEC>
cudaError_t launch_fixed_warp(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  constexpr int blk = gas::warp_block<G>();
  constexpr int smem = gas::warp_smem_bytes<KPT, G>();
  constexpr int arrays_per_block = (blk / 32) * (32 / G);
  auto k = gas::k_fixed_warp<KPT, G, VEC>;
  const cudaError_t e = cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
  if (e != cudaSuccess) return e;
  const int grid = persistent_grid_smem(k, blk, smem, (N + arrays_per_block - 1) / arrays_per_block);
  k<<<grid, blk, smem, s>>>(d, N, n, 1u);
  return cudaGetLastError();
}


template <int W, int WR, bool VEC>
cudaError_t launch_fixed_cta(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  auto k = gas::k_fixed_cta<W, WR, VEC>;
  constexpr int smem = gas::cta_smem_bytes<W, WR>();
  const cudaError_t e = cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
  if (e != cudaSuccess) return e;
  k<<<persistent_grid_smem(k, 32 * WR, smem, N), 32 * WR, smem, s>>>(d, N, n, 1u);
  return cudaGetLastError();
}

bool offsets512_bucket() {  // GAS_OFFSETS512=0: the (256, 512] offsets class on the network kernel
  const char* v = std::getenv("GAS_OFFSETS512");
  return !(v && std::strcmp(v, "0") == 0);
}

bool bucket_enabled() {
  const char* v = std::getenv("GAS_BUCKET");
  return !(v && std::strcmp(v, "0") == 0);
}

// Bucket-then-network, one array per CTA of W warps (bucket_cta.cuh).
template <int W, int WR, bool VEC>
cudaError_t launch_fixed_bucket_cta(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  auto k = gas::k_fixed_bucket_cta<W, WR, VEC>;
  constexpr int gr = gas::bkc_groups<WR>(), blk = gas::bkc_block<WR>();
  constexpr int smem = gas::BkCta<W, WR>::SMEM * gr;
  const cudaError_t e = cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
  if (e != cudaSuccess) return e;
  k<<<persistent_grid_smem(k, blk, smem, (N + gr - 1) / gr), blk, smem, s>>>(d, N, n, 1u);
  return cudaGetLastError();
}

template <int W, int WR, int RV = 16>
cudaError_t launch_offsets_bucket(uint32_t* d, const int64_t* off, int64_t N, int64_t lo, int64_t hi,
                                  unsigned long long* ctr, cudaStream_t s) {
  auto k = gas::k_offsets_bucket<W, WR, RV>;
  constexpr int gr = 1, blk = 32 * WR;
  constexpr int smem = gas::BkCta<W, WR>::SMEM * gr;
  const cudaError_t e = cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
  if (e != cudaSuccess) return e;
  k<<<persistent_grid_smem(k, blk, smem, ((N + 31) / 32 + gr - 1) / gr), blk, smem, s>>>(d, off, N, lo, hi, ctr, 1u);
  return cudaGetLastError();
}

// Fixed-length CTA classes (n > 1024): W warps' network, WR = ceil(n / 1024) real
// warps rounded to the instantiated set (padding blocks are virtual, see sort_cta).
template <bool VEC>
cudaError_t dispatch_fixed_cta(uint32_t* d, int64_t N, int n, cudaStream_t s) {
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

bool env_flag(const char* name) {
  const char* v = std::getenv(name);
  return v && v[0] != '\0' && std::strcmp(v, "0") != 0;
}

cudaError_t launch_fixed_1024_tma(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  // per-device attribute: set on every call (cheap), the current device may change
  const cudaError_t attr = cudaFuncSetAttribute(gas::k_fixed_1024_tma, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                                gas::kTmaSmemBytes);
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
  auto k = VEC ? gas::k_fixed_bucket1024 : gas::k_fixed_bucket1024_any<false>;
  const cudaError_t attr = cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, gas::kBkSmemBytes);
  if (attr != cudaSuccess) return attr;
  const int grid = persistent_grid_smem(k, gas::kBkBlock, gas::kBkSmemBytes,
                                        (N + gas::kBkBlock / 32 - 1) / (gas::kBkBlock / 32));
  k<<<grid, gas::kBkBlock, gas::kBkSmemBytes, s>>>(d, N, n, 1u);
  return cudaGetLastError();
}

// Bucket-then-network kernel for 256 < n <= 512 with aligned rows (bucket512.cuh).
cudaError_t launch_fixed_bucket512(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  const cudaError_t attr = cudaFuncSetAttribute(gas::k_fixed_bucket512, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                                gas::kBk5SmemBytes);
  if (attr != cudaSuccess) return attr;
  const int grid = persistent_grid_smem(gas::k_fixed_bucket512, gas::kBk5Block, gas::kBk5SmemBytes,
                                        (N + GAS_BK5_WARPS - 1) / GAS_BK5_WARPS);
  gas::k_fixed_bucket512<<<grid, gas::kBk5Block, gas::kBk5SmemBytes, s>>>(d, N, n, 1u);
  return cudaGetLastError();
}

template <bool VEC>
cudaError_t dispatch_fixed(uint32_t* d, int64_t N, int n, cudaStream_t s) {
  switch (size_class(n)) {
    case 2: return launch_fixed_warp<2, 1, false>(d, N, n, s);
    case 4: return launch_fixed_warp<4, 1, VEC>(d, N, n, s);
    case 8: return launch_fixed_warp<8, 1, VEC>(d, N, n, s);
    case 16: return launch_fixed_warp<16, 1, VEC>(d, N, n, s);
    case 32: return launch_fixed_warp<32, 1, VEC>(d, N, n, s);
    case 64: return launch_fixed_warp<32, 2, VEC>(d, N, n, s);
    case 128: return launch_fixed_warp<32, 4, VEC>(d, N, n, s);
    case 256: return launch_fixed_warp<32, 8, VEC>(d, N, n, s);
    case 512:
      if (VEC && bucket_enabled()) return launch_fixed_bucket512(d, N, n, s);
      return launch_fixed_warp<32, 16, VEC>(d, N, n, s);
    case 1024:
      // TMA-prefetch variant: opt-in (GAS_TMA=1). Measured on B200 it removes the
      // global-load stalls but is 5% slower overall (profiles/r01_ab_tma.txt):
      // the kernel is ALU/issue-bound, not latency-bound.
      if (VEC && env_flag("GAS_TMA")) return launch_fixed_1024_tma(d, N, n, s);
      if (bucket_enabled()) return launch_fixed_bucket1024<VEC>(d, N, n, s);
      return launch_fixed_warp<32, 32, VEC>(d, N, n, s);
    default: return dispatch_fixed_cta<VEC>(d, N, n, s);
  }
  return cudaErrorInvalidValue;
}

template <int KPT, int G>
cudaError_t launch_offsets_warp(uint32_t* d, const int64_t* off, int64_t N, cudaStream_t s) {
  constexpr int blk = gas::warp_block<G>();
  constexpr int smem = gas::warp_smem_bytes<KPT, G>();
  auto k = gas::k_offsets_warp<KPT, G>;
  const cudaError_t e = cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
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
  const cudaError_t e = cudaFuncSetAttribute(k, cudaFuncAttributeMaxDynamicSharedMemorySize, smem);
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

// GAS_CHECK=1 validation of CSR offsets: flag = 1 on any violation.
__global__ void k_check_offsets(const int64_t* __restrict__ off, int64_t N, int64_t max_len, int* flag) {
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < N; i += (int64_t)gridDim.x * blockDim.x) {
    const int64_t a = off[i], b = off[i + 1];
    if (a < 0 || b < a || b - a > max_len) atomicOr(flag, 1);
  }
}

// Device staging for gas_sort_arrays_host: streams and chunk buffers are created
// on first use and kept per device (re-used by later calls; grown on demand),
// so repeated host sorts do not pay cudaMalloc / cudaFree (which synchronises).
constexpr int kHostSlots = 4;
constexpr int kMaxDevices = 64;
struct HostStaging {
  std::mutex mu;
  cudaStream_t st[kHostSlots] = {};
  float* buf[kHostSlots] = {};
  int64_t bytes = 0;
  cudaError_t ensure(int slots, int64_t need) {
    cudaError_t e = cudaSuccess;
    for (int s = 0; s < kHostSlots && e == cudaSuccess; ++s)
      if (!st[s]) e = cudaStreamCreateWithFlags(&st[s], cudaStreamNonBlocking);
    if (e != cudaSuccess) return e;
    if (need > bytes) {
      for (int s = 0; s < kHostSlots; ++s)
        if (buf[s]) { cudaFree(buf[s]); buf[s] = nullptr; }
      bytes = need;
    }
    for (int s = 0; s < slots && e == cudaSuccess; ++s)
      if (!buf[s]) e = cudaMalloc(&buf[s], bytes);
    return e;
  }
};
HostStaging g_staging[kMaxDevices];

// Per-(device, caller stream) side streams of the offsets variant: the class
// launches fork over them and join back (see gas_sort_arrays_offsets).
constexpr int kMaxSide = 8;
struct SideStreams {
  cudaStream_t s[kMaxSide];
  cudaEvent_t fork, join[kMaxSide];
  std::mutex mu;
};
std::mutex g_side_mu;
std::map<std::pair<int, cudaStream_t>, SideStreams*> g_side;

int offsets_streams() {
  static const int k = [] {
    const char* v = std::getenv("GAS_OFFSETS_STREAMS");
    const int x = v ? std::atoi(v) : 8;
    return x < 1 ? 1 : (x > kMaxSide ? kMaxSide : x);
  }();
  return k;
}

cudaError_t side_streams_for(cudaStream_t stream, SideStreams** out) {
  int dev = 0;
  cudaError_t e = cudaGetDevice(&dev);
  if (e != cudaSuccess) return e;
  std::lock_guard<std::mutex> lock(g_side_mu);
  auto& slot = g_side[{dev, stream}];
  if (!slot) {
    SideStreams* ss = new SideStreams();
    e = cudaEventCreateWithFlags(&ss->fork, cudaEventDisableTiming);
    for (int i = 0; i < kMaxSide && e == cudaSuccess; ++i) {
      e = cudaStreamCreateWithFlags(&ss->s[i], cudaStreamNonBlocking);
      if (e == cudaSuccess) e = cudaEventCreateWithFlags(&ss->join[i], cudaEventDisableTiming);
    }
    if (e != cudaSuccess) return e;  // (leaks the partial set; only on a failing device)
    slot = ss;
  }
  *out = slot;
  return cudaSuccess;
}

// Per-(device, stream) window counters of the offsets variant (see there).
constexpr int kCounters = 9;
std::mutex g_ctr_mu;
std::map<std::pair<int, cudaStream_t>, unsigned long long*> g_ctr;

cudaError_t counters_for(cudaStream_t stream, unsigned long long** out) {
  int dev = 0;
  cudaError_t e = cudaGetDevice(&dev);
  if (e != cudaSuccess) return e;
  std::lock_guard<std::mutex> lock(g_ctr_mu);
  auto& slot = g_ctr[{dev, stream}];
  if (!slot) {
    e = cudaMalloc(&slot, kCounters * sizeof(unsigned long long));
    if (e != cudaSuccess) { slot = nullptr; return e; }
  }
  *out = slot;
  return cudaSuccess;
}

bool env_check() {
  const char* v = std::getenv("GAS_CHECK");
  return v && std::strcmp(v, "0") != 0 && v[0] != '\0';
}

}  // namespace

extern "C" {

gas_status gas_sort_arrays(float* d_data, int64_t num_arrays, int32_t array_len, cudaStream_t stream) {
  if (num_arrays < 0 || array_len < 0) return GAS_ERROR_INVALID_VALUE;
  if (num_arrays == 0 || array_len <= 1) return GAS_SUCCESS;
  if (array_len > kMaxLen) return GAS_ERROR_UNSUPPORTED;
  if (d_data == nullptr || (reinterpret_cast<uintptr_t>(d_data) & 3u)) return GAS_ERROR_INVALID_VALUE;
  uint32_t* d = reinterpret_cast<uint32_t*>(d_data);
  const bool vec = (reinterpret_cast<uintptr_t>(d_data) & 15u) == 0 && (array_len & 3) == 0;
  const cudaError_t e = vec ? dispatch_fixed<true>(d, num_arrays, array_len, stream)
                            : dispatch_fixed<false>(d, num_arrays, array_len, stream);
  if (e != cudaSuccess) return cuda_fail(e);
  g_launches.fetch_add(1, std::memory_order_relaxed);
  return GAS_SUCCESS;
}

gas_status gas_sort_arrays_offsets(float* d_data, const int64_t* d_offsets, int64_t num_arrays,
                                   int32_t max_array_len, cudaStream_t stream) {
  if (num_arrays < 0 || max_array_len < 0) return GAS_ERROR_INVALID_VALUE;
  if (max_array_len == 0) max_array_len = kMaxLen;
  if (max_array_len > kMaxLen) return GAS_ERROR_UNSUPPORTED;
  if (num_arrays == 0 || max_array_len <= 1) return GAS_SUCCESS;
  if (d_offsets == nullptr || (reinterpret_cast<uintptr_t>(d_offsets) & 7u)) return GAS_ERROR_INVALID_VALUE;
  if (d_data == nullptr || (reinterpret_cast<uintptr_t>(d_data) & 3u)) return GAS_ERROR_INVALID_VALUE;
  if (env_check()) {
    int* flag = nullptr;
    cudaError_t e = cudaMallocAsync(&flag, sizeof(int), stream);
    if (e != cudaSuccess) return cuda_fail(e);
    int h = 0;
    cudaMemsetAsync(flag, 0, sizeof(int), stream);
    k_check_offsets<<<num_sms() * 4, 256, 0, stream>>>(d_offsets, num_arrays, max_array_len, flag);
    g_launches.fetch_add(1, std::memory_order_relaxed);
    cudaMemcpyAsync(&h, flag, sizeof(int), cudaMemcpyDeviceToHost, stream);
    cudaFreeAsync(flag, stream);
    e = cudaStreamSynchronize(stream);
    if (e != cudaSuccess) return cuda_fail(e);
    if (h) return GAS_ERROR_INVALID_VALUE;
  }
  uint32_t* d = reinterpret_cast<uint32_t*>(d_data);
  // 9 window counters for the bucket classes' dynamic scheduling: 72 bytes per
  // (device, stream), allocated on first use and re-zeroed in stream order by
  // every call (calls on one stream are ordered; different streams never share)
  unsigned long long* ctr = nullptr;
  if (max_array_len > 256) {
    cudaError_t e = counters_for(stream, &ctr);
    if (e == cudaSuccess) e = cudaMemsetAsync(ctr, 0, kCounters * sizeof(unsigned long long), stream);
    if (e != cudaSuccess) return cuda_fail(e);
  }
  // size classes: 2, 4, ..., 2048 (len in (P/2, P]), then (2048, 3072] and (3072, 4096]
  const int32_t classes[] = {2, 4, 8, 16, 32, 64, 128, 256, 512, 1024, 2048, 3072, 4096, 6144, 8192, 12288, 16384};
  const int32_t lower[] = {1, 2, 4, 8, 16, 32, 64, 128, 256, 512, 1024, 2048, 3072, 4096, 6144, 8192, 12288};
  int nclass = 0;
  while (nclass < 17 && lower[nclass] < max_array_len) ++nclass;
  // The class launches are independent (disjoint arrays). With K > 1 they are
  // forked over K streams (largest classes first) so that each persistent
  // launch's last wave overlaps the next launches instead of idling SMs; the
  // caller's stream waits for all of them (CUDA-graph capture follows the
  // fork/join). GAS_OFFSETS_STREAMS=1 restores one stream.
  SideStreams* ss = nullptr;
  if (offsets_streams() > 1 && nclass > 1) {
    const cudaError_t e = side_streams_for(stream, &ss);
    if (e != cudaSuccess) return cuda_fail(e);
  }
  if (!ss) {
    for (int c = 0; c < nclass; ++c) {
      const cudaError_t e = dispatch_offsets_class(classes[c], d, d_offsets, num_arrays, ctr, stream);
      if (e != cudaSuccess) return cuda_fail(e);
      g_launches.fetch_add(1, std::memory_order_relaxed);
    }
    return GAS_SUCCESS;
  }
  std::lock_guard<std::mutex> lock(ss->mu);
  const int K = offsets_streams();
  cudaError_t e = cudaEventRecord(ss->fork, stream);
  for (int i = 0; i < K && e == cudaSuccess; ++i) e = cudaStreamWaitEvent(ss->s[i], ss->fork, 0);
  for (int c = nclass - 1, i = 0; c >= 0 && e == cudaSuccess; --c, ++i) {
    e = dispatch_offsets_class(classes[c], d, d_offsets, num_arrays, ctr, ss->s[i % K]);
    if (e == cudaSuccess) g_launches.fetch_add(1, std::memory_order_relaxed);
  }
  // always join (also after an error) so that the caller's stream never races ahead
  for (int i = 0; i < K; ++i) {
    const cudaError_t r = cudaEventRecord(ss->join[i], ss->s[i]);
    const cudaError_t w = r == cudaSuccess ? cudaStreamWaitEvent(stream, ss->join[i], 0) : r;
    if (e == cudaSuccess) e = w;
  }
  return e == cudaSuccess ? GAS_SUCCESS : cuda_fail(e);
}

gas_status gas_sort_pairs(float* d_keys, uint32_t* d_values, int64_t num_arrays, int32_t array_len,
                          cudaStream_t stream) {
  if (num_arrays < 0 || array_len < 0) return GAS_ERROR_INVALID_VALUE;
  if (num_arrays == 0 || array_len <= 1) return GAS_SUCCESS;
  if (array_len > kMaxPairsLen) return GAS_ERROR_UNSUPPORTED;
  if (d_keys == nullptr || d_values == nullptr || (reinterpret_cast<uintptr_t>(d_keys) & 3u) ||
      (reinterpret_cast<uintptr_t>(d_values) & 3u))
    return GAS_ERROR_INVALID_VALUE;
  const cudaError_t e = dispatch_pairs(reinterpret_cast<uint32_t*>(d_keys), d_values, num_arrays, array_len, stream);
  if (e != cudaSuccess) return cuda_fail(e);
  g_launches.fetch_add(1, std::memory_order_relaxed);
  return GAS_SUCCESS;
}

gas_status gas_sort_arrays_host(float* h_data, int64_t num_arrays, int32_t array_len) {
  if (num_arrays < 0 || array_len < 0) return GAS_ERROR_INVALID_VALUE;
  if (num_arrays == 0 || array_len <= 1) return GAS_SUCCESS;
  if (array_len > kMaxLen) return GAS_ERROR_UNSUPPORTED;
  if (h_data == nullptr || (reinterpret_cast<uintptr_t>(h_data) & 3u)) return GAS_ERROR_INVALID_VALUE;
  const char* env_chunk = std::getenv("GAS_HOST_CHUNK_MB");  // tuning knob (default 128 MB)
  const char* env_slots = std::getenv("GAS_HOST_SLOTS");     // 1..4 (default 3)
  const int64_t chunk_bytes = (env_chunk ? std::atoll(env_chunk) : 128ll) << 20;
  const int want_slots = env_slots ? std::atoi(env_slots) : 3;
  const int64_t row = (int64_t)array_len * 4;
  int64_t per_chunk = chunk_bytes / row;
  if (per_chunk < 1) per_chunk = 1;
  if (per_chunk > num_arrays) per_chunk = num_arrays;
  const int64_t nchunks = (num_arrays + per_chunk - 1) / per_chunk;
  int slots = (int)(nchunks < want_slots ? nchunks : want_slots);
  if (slots > kHostSlots) slots = kHostSlots;
  if (slots < 1) slots = 1;
  int dev = 0;
  cudaError_t e = cudaGetDevice(&dev);
  if (e != cudaSuccess) return cuda_fail(e);
  if (dev < 0 || dev >= kMaxDevices) return GAS_ERROR_UNSUPPORTED;
  HostStaging& hs = g_staging[dev];
  std::lock_guard<std::mutex> lock(hs.mu);  // one host-path sort per device at a time (they share PCIe anyway)
  e = hs.ensure(slots, per_chunk * row);
  if (e != cudaSuccess) return cuda_fail(e);
  gas_status status = GAS_SUCCESS;
  for (int64_t c = 0; c < nchunks && e == cudaSuccess && status == GAS_SUCCESS; ++c) {
    const int sl = (int)(c % slots);
    const int64_t first = c * per_chunk;
    const int64_t cnt = (first + per_chunk <= num_arrays) ? per_chunk : num_arrays - first;
    float* h = h_data + first * array_len;
    e = cudaMemcpyAsync(hs.buf[sl], h, cnt * row, cudaMemcpyHostToDevice, hs.st[sl]);
    if (e != cudaSuccess) break;
    status = gas_sort_arrays(hs.buf[sl], cnt, array_len, hs.st[sl]);
    if (status != GAS_SUCCESS) break;
    e = cudaMemcpyAsync(h, hs.buf[sl], cnt * row, cudaMemcpyDeviceToHost, hs.st[sl]);
  }
  for (int sl = 0; sl < slots; ++sl) {
    const cudaError_t e2 = cudaStreamSynchronize(hs.st[sl]);
    if (e == cudaSuccess) e = e2;
  }
  if (status != GAS_SUCCESS) return status;
  if (e != cudaSuccess) return cuda_fail(e);
  return GAS_SUCCESS;
}

int32_t gas_max_array_len(void) { return kMaxLen; }

const char* gas_status_string(gas_status s) {
  switch (s) {
    case GAS_SUCCESS: return "GAS_SUCCESS";
    case GAS_ERROR_INVALID_VALUE: return "GAS_ERROR_INVALID_VALUE";
    case GAS_ERROR_UNSUPPORTED: return "GAS_ERROR_UNSUPPORTED";
    case GAS_ERROR_CUDA: return "GAS_ERROR_CUDA";
  }
  return "GAS_UNKNOWN_STATUS";
}

int gas_last_cuda_error(void) { return g_last_cuda_error; }

int64_t gas_launch_count(void) { return g_launches.load(std::memory_order_relaxed); }

}  // extern "C"
