// gasgen.cu — device twin of datagen/__init__.py (recipe in gasgen.h).
// Bench/test support, not part of the sort: no ordering arithmetic here.
#include "gasgen.h"

namespace {

__device__ __forceinline__ uint64_t mix(uint64_t z) {
  z ^= z >> 30; z *= 0xBF58476D1CE4E5B9ull;
  z ^= z >> 27; z *= 0x94D049BB133111EBull;
  return z ^ (z >> 31);
}
constexpr uint64_t G = 0x9E3779B97F4A7C15ull;

__device__ __forceinline__ uint64_t h3(uint64_t s, uint64_t i, uint64_t j) {
  return mix(mix(s ^ ((i + 1) * G)) + (j + 1) * G);
}

__device__ __forceinline__ uint32_t value(int dist, uint64_t s, uint64_t i, uint64_t j, uint64_t n) {
  const uint64_t h = h3(s, i, j);
  const uint32_t hi = (uint32_t)(h >> 32), lo = (uint32_t)h;
  switch (dist) {
    case 0: return __float_as_uint(__uint2float_rn(hi >> 1));
    case 1: return hi;
    case 2: return ((127u + __popc(lo & 0xFFFFu)) << 23) | (hi >> 9);
    case 3: return __float_as_uint(__fadd_rn(100.0f, __fmul_rn(__uint2float_rn(hi >> 8), 1900.0f / 16777216.0f)));
    case 4: return __float_as_uint(__uint2float_rn(hi >> 28));
    case 5:
    case 6: {
      const uint32_t b = (uint32_t)(h3(s, i, 0xFFFFFFFFull) >> 41);
      const uint32_t k = dist == 5 ? (uint32_t)j : (uint32_t)(n - 1 - j);
      return __float_as_uint(__uint2float_rn(b + k));
    }
    case 7: {
      const uint32_t c = lo % 1000u, sign = hi & 0x80000000u;
      if (c < 100u) return 0x80000000u;
      if (c < 200u) return 0u;
      if (c < 225u) return 0x7F800000u;
      if (c < 250u) return 0xFF800000u;
      if (c < 300u) return sign | 0x7F800000u | (((hi >> 30) & 1u) << 22) | ((hi & 0x3FFFFFu) | 1u);
      if (c < 320u) return sign | ((hi & 0x7FFFFFu) | 1u);
      return __float_as_uint(__fmul_rn(__int2float_rn((int32_t)hi), 1000.0f / 2147483648.0f));
    }
    default: return 0u;
  }
}

__global__ void k_fixed(uint32_t* __restrict__ d, int dist, uint64_t seed, int64_t i0, int64_t N, int32_t n) {
  const int64_t total = N * (int64_t)n;
  for (int64_t e = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; e < total;
       e += (int64_t)gridDim.x * blockDim.x) {
    const int64_t i = e / n, j = e - i * n;
    d[e] = value(dist, seed, (uint64_t)(i0 + i), (uint64_t)j, (uint64_t)n);
  }
}

__global__ void k_ragged(uint32_t* __restrict__ d, const int64_t* __restrict__ off, int dist, uint64_t seed,
                         int64_t i0, int64_t N) {
  const int lane = threadIdx.x & 31;
  const int64_t warps = (int64_t)gridDim.x * (blockDim.x >> 5);
  const int64_t base = off[0];
  for (int64_t k = blockIdx.x * (int64_t)(blockDim.x >> 5) + (threadIdx.x >> 5); k < N; k += warps) {
    const int64_t a = off[k], len = off[k + 1] - a;
    for (int64_t j = lane; j < len; j += 32)
      d[a - base + j] = value(dist, seed, (uint64_t)(i0 + k), (uint64_t)j, (uint64_t)len);
  }
}

}  // namespace

extern "C" int gasgen_fixed(uint32_t* d, int dist, uint64_t seed, int64_t i0, int64_t N, int32_t n,
                            cudaStream_t stream) {
  if (N <= 0 || n <= 0) return 0;
  int dev = 0, sms = 148;
  cudaGetDevice(&dev);
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
  k_fixed<<<sms * 8, 256, 0, stream>>>(d, dist, seed, i0, N, n);
  return (int)cudaGetLastError();
}

extern "C" int gasgen_ragged(uint32_t* d, const int64_t* d_off, int dist, uint64_t seed, int64_t i0,
                             int64_t N, cudaStream_t stream) {
  if (N <= 0) return 0;
  int dev = 0, sms = 148;
  cudaGetDevice(&dev);
  cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
  k_ragged<<<sms * 8, 256, 0, stream>>>(d, d_off, dist, seed, i0, N);
  return (int)cudaGetLastError();
}
