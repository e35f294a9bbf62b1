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
#include "launch_util.cuh"

namespace {

constexpr int32_t kMaxPairsLen = 8192;  // 64-bit network elements: 8 KB of SMEM per 1024
constexpr int32_t kMaxLen = 65536;       // fixed-length arrays: 16x the spectra bound of P:L170-173
constexpr int32_t kMaxOffsetsLen = 16384;  // variable-length classes (one CTA per array)

thread_local int g_last_cuda_error = 0;

gas_status cuda_fail(cudaError_t e) {
  g_last_cuda_error = (int)e;
  return GAS_ERROR_CUDA;
}

using namespace gas_host;

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
  // offsets staging of gas_sort_arrays_offsets_host: pinned host + device, per slot
  int64_t* off_h[kHostSlots] = {};
  int64_t* off_d[kHostSlots] = {};
  int64_t off_cap = 0;  // entries
  cudaError_t ensure_offsets(int slots, int64_t entries) {
    cudaError_t e = cudaSuccess;
    if (entries > off_cap) {
      for (int s = 0; s < kHostSlots; ++s) {
        if (off_h[s]) { cudaFreeHost(off_h[s]); off_h[s] = nullptr; }
        if (off_d[s]) { cudaFree(off_d[s]); off_d[s] = nullptr; }
      }
      off_cap = entries;
    }
    for (int s = 0; s < slots && e == cudaSuccess; ++s) {
      if (!off_h[s]) e = cudaMallocHost(&off_h[s], off_cap * sizeof(int64_t));
      if (e == cudaSuccess && !off_d[s]) e = cudaMalloc(&off_d[s], off_cap * sizeof(int64_t));
    }
    return e;
  }
};
HostStaging g_staging[kMaxDevices];

// Per-(device, caller stream) side streams of the offsets variant: the class
// launches fork over them and join back (see gas_sort_arrays_offsets). At most
// kMaxSideSets caller streams get a set (8 streams + 9 events each); calls on
// further streams launch every class on the caller's stream.
// gas_release_stream() destroys a stream's set.
constexpr int kMaxSide = 8;
constexpr size_t kMaxSideSets = 64;
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

void destroy_side(SideStreams* ss) {
  for (int i = 0; i < kMaxSide; ++i) {
    if (ss->s[i]) cudaStreamDestroy(ss->s[i]);
    if (ss->join[i]) cudaEventDestroy(ss->join[i]);
  }
  if (ss->fork) cudaEventDestroy(ss->fork);
  delete ss;
}

// *out = nullptr (and success) when the cache is full: the caller then uses one stream.
cudaError_t side_streams_for(cudaStream_t stream, SideStreams** out) {
  *out = nullptr;
  int dev = 0;
  cudaError_t e = cudaGetDevice(&dev);
  if (e != cudaSuccess) return e;
  std::lock_guard<std::mutex> lock(g_side_mu);
  auto it = g_side.find({dev, stream});
  if (it != g_side.end()) {
    *out = it->second;
    return cudaSuccess;
  }
  if (g_side.size() >= kMaxSideSets) return cudaSuccess;
  SideStreams* ss = new SideStreams();
  for (int i = 0; i < kMaxSide; ++i) { ss->s[i] = nullptr; ss->join[i] = nullptr; }
  ss->fork = nullptr;
  e = cudaEventCreateWithFlags(&ss->fork, cudaEventDisableTiming);
  for (int i = 0; i < kMaxSide && e == cudaSuccess; ++i) {
    e = cudaStreamCreateWithFlags(&ss->s[i], cudaStreamNonBlocking);
    if (e == cudaSuccess) e = cudaEventCreateWithFlags(&ss->join[i], cudaEventDisableTiming);
  }
  if (e != cudaSuccess) {
    destroy_side(ss);
    return e;
  }
  g_side[{dev, stream}] = ss;
  *out = ss;
  return cudaSuccess;
}

// Window counters of the offsets variant's dynamic scheduling: 9 x 8 bytes
// per call, stream-ordered from the library's memory pool (each call and each
// captured graph owns its counters: concurrent calls never share them).
constexpr int kCounters = 9;

bool env_check() {
  const char* v = std::getenv("GAS_CHECK");
  return v && std::strcmp(v, "0") != 0 && v[0] != '\0';
}

}  // namespace

namespace gas_host {

// The variable-length (CSR) sort: per-class launches forked over side streams.
cudaError_t offsets_sort(uint32_t* d, const int64_t* off, int64_t N, int32_t max_len, cudaStream_t s) {
  // 9 window counters for the bucket classes' dynamic scheduling (72 bytes per call)
  unsigned long long* ctr = nullptr;
  if (max_len > 256) {
    void* p = nullptr;
    cudaError_t e = ws_alloc(&p, kCounters * sizeof(unsigned long long), s);
    if (e == cudaSuccess) e = cudaMemsetAsync(p, 0, kCounters * sizeof(unsigned long long), s);
    if (e != cudaSuccess) return e;
    ctr = static_cast<unsigned long long*>(p);
  }
  // every exit below frees the counters on `s`, after the work that uses them
  auto release = [&](cudaError_t e) -> cudaError_t {
    if (ctr) {
      const cudaError_t f = cudaFreeAsync(ctr, s);
      if (e == cudaSuccess) e = f;
    }
    return e;
  };
  // size classes: 2, 4, ..., 2048 (len in (P/2, P]), then (2048, 3072] and (3072, 4096]
  const int32_t classes[] = {2, 4, 8, 16, 32, 64, 128, 256, 512, 1024, 2048, 3072, 4096, 6144, 8192, 12288, 16384};
  const int32_t lower[] = {1, 2, 4, 8, 16, 32, 64, 128, 256, 512, 1024, 2048, 3072, 4096, 6144, 8192, 12288};
  int nclass = 0;
  while (nclass < 17 && lower[nclass] < max_len) ++nclass;
  // The class launches are independent (disjoint arrays). With K > 1 they are
  // forked over K streams (largest classes first) so that each persistent
  // launch's last wave overlaps the next launches instead of idling SMs; the
  // caller's stream waits for all of them (CUDA-graph capture follows the
  // fork/join). GAS_OFFSETS_STREAMS=1 restores one stream.
  SideStreams* ss = nullptr;
  if (offsets_streams() > 1 && nclass > 1) {
    const cudaError_t e = side_streams_for(s, &ss);
    if (e != cudaSuccess) return release(e);
  }
  if (!ss) {
    for (int c = 0; c < nclass; ++c) {
      const cudaError_t e = dispatch_offsets_class(classes[c], d, off, N, ctr, s);
      if (e != cudaSuccess) return release(e);
      launch_counter() += 1;
    }
    return release(cudaSuccess);
  }
  std::lock_guard<std::mutex> lock(ss->mu);
  const int K = offsets_streams();
  cudaError_t e = cudaEventRecord(ss->fork, s);
  for (int i = 0; i < K && e == cudaSuccess; ++i) e = cudaStreamWaitEvent(ss->s[i], ss->fork, 0);
  for (int c = nclass - 1, i = 0; c >= 0 && e == cudaSuccess; --c, ++i) {
    e = dispatch_offsets_class(classes[c], d, off, N, ctr, ss->s[i % K]);
    if (e == cudaSuccess) launch_counter() += 1;
  }
  // always join (also after an error) so that the caller's stream never races ahead
  for (int i = 0; i < K; ++i) {
    const cudaError_t r = cudaEventRecord(ss->join[i], ss->s[i]);
    const cudaError_t w = r == cudaSuccess ? cudaStreamWaitEvent(s, ss->join[i], 0) : r;
    if (e == cudaSuccess) e = w;
  }
  return release(e);
}

}  // namespace gas_host

extern "C" {

gas_status gas_sort_arrays(float* d_data, int64_t num_arrays, int32_t array_len, cudaStream_t stream) {
  if (num_arrays < 0 || array_len < 0) return GAS_ERROR_INVALID_VALUE;
  if (num_arrays == 0 || array_len <= 1) return GAS_SUCCESS;
  if (array_len > kMaxLen) return GAS_ERROR_UNSUPPORTED;
  if (d_data == nullptr || (reinterpret_cast<uintptr_t>(d_data) & 3u)) return GAS_ERROR_INVALID_VALUE;
  uint32_t* d = reinterpret_cast<uint32_t*>(d_data);
  const bool vec = (reinterpret_cast<uintptr_t>(d_data) & 15u) == 0 && (array_len & 3) == 0;
  const cudaError_t e = array_len <= 512     ? dispatch_fixed_small(vec, d, num_arrays, array_len, stream)
                        : array_len <= 1024  ? dispatch_fixed_1024(vec, d, num_arrays, array_len, stream)
                        : array_len <= 16384 ? dispatch_fixed_cta(vec, d, num_arrays, array_len, stream)
                                             : dispatch_fixed_cluster(vec, d, num_arrays, array_len, stream);
  if (e != cudaSuccess) return cuda_fail(e);
  if (array_len <= 512 || (array_len > 1024 && array_len <= 16384)) launch_counter() += 1;  // others count their own
  return GAS_SUCCESS;
}

gas_status gas_sort_arrays_offsets(float* d_data, const int64_t* d_offsets, int64_t num_arrays,
                                   int32_t max_array_len, cudaStream_t stream) {
  if (num_arrays < 0 || max_array_len < 0) return GAS_ERROR_INVALID_VALUE;
  if (max_array_len == 0) max_array_len = kMaxOffsetsLen;
  if (max_array_len > kMaxOffsetsLen) return GAS_ERROR_UNSUPPORTED;
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
    launch_counter() += 1;
    cudaMemcpyAsync(&h, flag, sizeof(int), cudaMemcpyDeviceToHost, stream);
    cudaFreeAsync(flag, stream);
    e = cudaStreamSynchronize(stream);
    if (e != cudaSuccess) return cuda_fail(e);
    if (h) return GAS_ERROR_INVALID_VALUE;
  }
  const cudaError_t e = offsets_sort(reinterpret_cast<uint32_t*>(d_data), d_offsets, num_arrays, max_array_len, stream);
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
  launch_counter() += 1;
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

gas_status gas_sort_arrays_offsets_host(float* h_data, const int64_t* h_offsets, int64_t num_arrays,
                                        int32_t max_array_len) {
  if (num_arrays < 0 || max_array_len < 0) return GAS_ERROR_INVALID_VALUE;
  if (max_array_len == 0) max_array_len = kMaxOffsetsLen;
  if (max_array_len > kMaxOffsetsLen) return GAS_ERROR_UNSUPPORTED;
  if (num_arrays == 0 || max_array_len <= 1) return GAS_SUCCESS;
  if (h_offsets == nullptr || h_data == nullptr || (reinterpret_cast<uintptr_t>(h_data) & 3u))
    return GAS_ERROR_INVALID_VALUE;
  const char* env_chunk = std::getenv("GAS_HOST_CHUNK_MB");
  const char* env_slots = std::getenv("GAS_HOST_SLOTS");
  const int64_t chunk_elems = ((env_chunk ? std::atoll(env_chunk) : 128ll) << 20) / 4;
  const int64_t max_chunk_arrays = 1 << 20;  // bounds the offsets staging (8 MB per slot)
  int slots = env_slots ? std::atoi(env_slots) : 3;
  slots = slots < 1 ? 1 : (slots > kHostSlots ? kHostSlots : slots);
  int dev = 0;
  cudaError_t e = cudaGetDevice(&dev);
  if (e != cudaSuccess) return cuda_fail(e);
  if (dev < 0 || dev >= kMaxDevices) return GAS_ERROR_UNSUPPORTED;
  HostStaging& hs = g_staging[dev];
  std::lock_guard<std::mutex> lock(hs.mu);
  const int64_t per = chunk_elems > max_array_len ? chunk_elems : max_array_len;
  e = hs.ensure(slots, per * 4);
  if (e == cudaSuccess) e = hs.ensure_offsets(slots, max_chunk_arrays + 1);
  if (e != cudaSuccess) return cuda_fail(e);
  gas_status status = GAS_SUCCESS;
  int64_t a = 0;
  for (int64_t c = 0; a < num_arrays && e == cudaSuccess && status == GAS_SUCCESS; ++c) {
    // chunk = arrays [a, b): whole arrays, at most `per` elements and max_chunk_arrays arrays
    int64_t b = a + 1;
    while (b < num_arrays && b - a < max_chunk_arrays && h_offsets[b + 1] - h_offsets[a] <= per) ++b;
    const int sl = (int)(c % slots);
    e = cudaStreamSynchronize(hs.st[sl]);  // the slot's previous chunk is done with its staging
    if (e != cudaSuccess) break;
    const int64_t base = h_offsets[a], elems = h_offsets[b] - base;
    if (elems < 0 || elems > per) { status = GAS_ERROR_INVALID_VALUE; break; }
    std::memcpy(hs.off_h[sl], h_offsets + a, (b - a + 1) * sizeof(int64_t));
    e = cudaMemcpyAsync(hs.off_d[sl], hs.off_h[sl], (b - a + 1) * sizeof(int64_t), cudaMemcpyHostToDevice, hs.st[sl]);
    if (e == cudaSuccess && elems > 0)
      e = cudaMemcpyAsync(hs.buf[sl], h_data + base, elems * 4, cudaMemcpyHostToDevice, hs.st[sl]);
    if (e != cudaSuccess) break;
    // the device offsets are the caller's (not rebased): the data pointer is shifted instead
    status = gas_sort_arrays_offsets(hs.buf[sl] - base, hs.off_d[sl], b - a, max_array_len, hs.st[sl]);
    if (status != GAS_SUCCESS) break;
    if (elems > 0) e = cudaMemcpyAsync(h_data + base, hs.buf[sl], elems * 4, cudaMemcpyDeviceToHost, hs.st[sl]);
    a = b;
  }
  for (int sl = 0; sl < slots; ++sl) {
    const cudaError_t e2 = cudaStreamSynchronize(hs.st[sl]);
    if (e == cudaSuccess) e = e2;
  }
  if (status != GAS_SUCCESS) return status;
  if (e != cudaSuccess) return cuda_fail(e);
  return GAS_SUCCESS;
}

gas_status gas_release_stream(cudaStream_t stream) {
  int dev = 0;
  const cudaError_t e = cudaGetDevice(&dev);
  if (e != cudaSuccess) return cuda_fail(e);
  SideStreams* ss = nullptr;
  {
    std::lock_guard<std::mutex> lock(g_side_mu);
    auto it = g_side.find({dev, stream});
    if (it == g_side.end()) return GAS_SUCCESS;
    ss = it->second;
    g_side.erase(it);
  }
  {
    std::lock_guard<std::mutex> lock(ss->mu);  // a call still enqueueing on this set finishes first
  }
  for (int i = 0; i < kMaxSide; ++i)
    if (ss->s[i]) cudaStreamSynchronize(ss->s[i]);
  destroy_side(ss);
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

int64_t gas_launch_count(void) { return launch_counter().load(std::memory_order_relaxed); }

}  // extern "C"
