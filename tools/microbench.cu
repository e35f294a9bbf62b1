// Throughput microbenchmarks for the instruction mix of an in-register
// sorting network on sm_100a: integer min/max,
// predicated min/max, IADD3, IMAD, LOP3, SHFL, LDS/STS, plus a streaming
// copy that gives the achievable HBM bandwidth for a 1-read + 1-write kernel.
//
// Build: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o microbench microbench.cu
// Prints one JSON object.
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

#define CK(x) do { cudaError_t e = (x); if (e != cudaSuccess) { \
  fprintf(stderr, "%s:%d %s\n", __FILE__, __LINE__, cudaGetErrorString(e)); return 1; } } while (0)

constexpr int CHAINS = 8;
constexpr int ITERS = 4096;

struct Res { unsigned long long cycles; };

// Each op kernel: CHAINS independent dependency chains per thread, ITERS
// iterations; per-block cycle count measured with clock64 by thread 0.
#define OPKERNEL(NAME, ...)                                                    \
__global__ void __launch_bounds__(1024) NAME(uint32_t* out, unsigned long long* cyc, uint32_t seed) { \
  uint32_t x[CHAINS], y[CHAINS];                                               \
  _Pragma("unroll") for (int c = 0; c < CHAINS; ++c) {                         \
    x[c] = seed * (threadIdx.x + 1) + c * 977u; y[c] = seed ^ (c * 131u + threadIdx.x); } \
  bool pr = (threadIdx.x & 1);                                                 \
  __syncthreads();                                                             \
  unsigned long long t0 = clock64();                                           \
  for (int it = 0; it < ITERS; ++it) {                                         \
    _Pragma("unroll") for (int c = 0; c < CHAINS; ++c) { __VA_ARGS__; }        \
  }                                                                            \
  __syncthreads();                                                             \
  unsigned long long t1 = clock64();                                           \
  uint32_t acc = 0;                                                            \
  _Pragma("unroll") for (int c = 0; c < CHAINS; ++c) acc += x[c] + y[c];       \
  out[blockIdx.x * blockDim.x + threadIdx.x] = acc + pr;                       \
  if (threadIdx.x == 0) cyc[blockIdx.x] = t1 - t0;                             \
}

// 2 ops per chain-iteration so that x and y both stay live.
OPKERNEL(k_min_u32, { uint32_t a = x[c], b = y[c];
  asm volatile("min.u32 %0, %1, %2;" : "=r"(x[c]) : "r"(a), "r"(b));
  asm volatile("max.u32 %0, %1, %2;" : "=r"(y[c]) : "r"(a), "r"(b)); })
OPKERNEL(k_minmax_pred, { uint32_t a = x[c], b = y[c];
  x[c] = pr ? max(a, b) : min(a, b); y[c] = pr ? min(a, b) ^ 1u : max(a, b) ^ 1u; })
OPKERNEL(k_iadd3, { uint32_t a = x[c], b = y[c];
  asm volatile("add.u32 %0, %1, %2;" : "=r"(x[c]) : "r"(a), "r"(b));
  asm volatile("sub.u32 %0, %1, %2;" : "=r"(y[c]) : "r"(a), "r"(b)); })
OPKERNEL(k_imad, { uint32_t a = x[c], b = y[c];
  asm volatile("mad.lo.u32 %0, %1, %2, %3;" : "=r"(x[c]) : "r"(a), "r"(b), "r"(a));
  asm volatile("mad.lo.u32 %0, %1, %2, %3;" : "=r"(y[c]) : "r"(b), "r"(a), "r"(b)); })
OPKERNEL(k_lop3, { uint32_t a = x[c], b = y[c];
  asm volatile("xor.b32 %0, %1, %2;" : "=r"(x[c]) : "r"(a), "r"(b));
  asm volatile("and.b32 %0, %1, %2;" : "=r"(y[c]) : "r"(a), "r"(b)); })
OPKERNEL(k_fmnmx, { float a = __uint_as_float(x[c]), b = __uint_as_float(y[c]); float r0, r1;
  asm volatile("min.f32 %0, %1, %2;" : "=f"(r0) : "f"(a), "f"(b));
  asm volatile("max.f32 %0, %1, %2;" : "=f"(r1) : "f"(a), "f"(b));
  x[c] = __float_as_uint(r0); y[c] = __float_as_uint(r1); })
OPKERNEL(k_min3, { uint32_t a = x[c], b = y[c];
  x[c] = __vimin3_u32(a, b, x[(c + 1) % CHAINS]); y[c] = __vimax3_u32(a, b, y[(c + 1) % CHAINS]); })
OPKERNEL(k_shfl, { uint32_t a = x[c], b = y[c];
  x[c] = __shfl_xor_sync(0xffffffffu, a, 1 + (c & 15)); y[c] = __shfl_xor_sync(0xffffffffu, b, 16 >> (c & 3)); })
// Mixed compare-exchange: min on ALU, max recomputed as a+b-min on the FMA pipe.
OPKERNEL(k_ce_mixed, { uint32_t a = x[c], b = y[c]; uint32_t mn, s, mx;
  asm volatile("min.u32 %0, %1, %2;" : "=r"(mn) : "r"(a), "r"(b));
  asm volatile("mad.lo.u32 %0, %1, 1, %2;" : "=r"(s) : "r"(a), "r"(b));
  asm volatile("mad.lo.u32 %0, %1, -1, %2;" : "=r"(mx) : "r"(mn), "r"(s));
  x[c] = mn; y[c] = mx; })

__global__ void __launch_bounds__(1024) k_smem(uint32_t* out, unsigned long long* cyc, uint32_t seed) {
  __shared__ uint32_t s[8192];
  for (int i = threadIdx.x; i < 8192; i += blockDim.x) s[i] = i * seed;
  __syncthreads();
  uint32_t acc = 0;
  uint32_t idx = threadIdx.x;
  unsigned long long t0 = clock64();
  for (int it = 0; it < ITERS; ++it) {
#pragma unroll
    for (int c = 0; c < CHAINS; ++c) {
      uint32_t v = s[(idx + c * 1024) & 8191];
      s[(idx + c * 1024 + 32) & 8191] = v + 1;
      acc += v;
    }
    idx += 1;
  }
  __syncthreads();
  unsigned long long t1 = clock64();
  out[blockIdx.x * blockDim.x + threadIdx.x] = acc;
  if (threadIdx.x == 0) cyc[blockIdx.x] = t1 - t0;
}

__global__ void copy_v4(const uint4* __restrict__ a, uint4* __restrict__ b, size_t n) {
  size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x;
  size_t stride = (size_t)gridDim.x * blockDim.x;
  for (; i < n; i += stride) b[i] = a[i];
}

// in-place read-modify-write (same footprint pattern as an in-place sort)
__global__ void rmw_v4(uint4* __restrict__ a, size_t n) {
  size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x;
  size_t stride = (size_t)gridDim.x * blockDim.x;
  for (; i < n; i += stride) { uint4 v = a[i]; v.x ^= 1u; a[i] = v; }
}

typedef void (*OpK)(uint32_t*, unsigned long long*, uint32_t);

int main() {
  cudaDeviceProp p;
  CK(cudaGetDeviceProperties(&p, 0));
  int clk_khz = 0, memclk_khz = 0;
  cudaDeviceGetAttribute(&clk_khz, cudaDevAttrClockRate, 0);
  cudaDeviceGetAttribute(&memclk_khz, cudaDevAttrMemoryClockRate, 0);
  printf("{\"name\": \"%s\", \"sm\": %d, \"cc\": \"%d.%d\", \"smem_per_sm\": %zu, \"smem_optin\": %zu, "
         "\"l2\": %d, \"regs_per_sm\": %d, \"hbm_bytes\": %zu, \"clock_khz\": %d, \"memclock_khz\": %d, "
         "\"bus_bits\": %d,\n", p.name, p.multiProcessorCount, p.major, p.minor,
         p.sharedMemPerMultiprocessor, p.sharedMemPerBlockOptin, p.l2CacheSize, p.regsPerMultiprocessor,
         p.totalGlobalMem, clk_khz, memclk_khz, p.memoryBusWidth);
  int nsm = p.multiProcessorCount;
  uint32_t* out; unsigned long long* cyc;
  CK(cudaMalloc(&out, nsm * 1024 * 4 * 4));
  CK(cudaMalloc(&cyc, nsm * 4 * sizeof(unsigned long long)));
  struct { const char* name; OpK k; double ops_per_chain_iter; } ks[] = {
    {"min_max_u32", k_min_u32, 2}, {"minmax_pred", k_minmax_pred, 2}, {"iadd", k_iadd3, 2},
    {"imad", k_imad, 2}, {"lop", k_lop3, 2}, {"fmnmx", k_fmnmx, 2}, {"min3_max3", k_min3, 2},
    {"shfl", k_shfl, 2}, {"ce_mixed_ce", k_ce_mixed, 1}, {"lds_sts_pair", k_smem, 1},
  };
  printf("\"ops_per_clk_per_sm\": {");
  for (size_t q = 0; q < sizeof(ks) / sizeof(ks[0]); ++q) {
    ks[q].k<<<nsm, 1024>>>(out, cyc, 12345u);  // warm
    CK(cudaDeviceSynchronize());
    ks[q].k<<<nsm, 1024>>>(out, cyc, 777u);
    CK(cudaDeviceSynchronize());
    unsigned long long h[1024];
    CK(cudaMemcpy(h, cyc, nsm * sizeof(unsigned long long), cudaMemcpyDeviceToHost));
    double mx = 0; for (int i = 0; i < nsm; ++i) mx = h[i] > mx ? h[i] : mx;
    double ops = 1024.0 * ITERS * CHAINS * ks[q].ops_per_chain_iter;
    printf("%s\"%s\": %.2f", q ? ", " : "", ks[q].name, ops / mx);
  }
  printf("},\n");
  // bandwidth
  size_t bytes = (size_t)4 << 30;  // 4 GiB per buffer
  uint4 *a, *b;
  CK(cudaMalloc(&a, bytes)); CK(cudaMalloc(&b, bytes));
  CK(cudaMemset(a, 1, bytes)); CK(cudaMemset(b, 2, bytes));
  size_t n = bytes / 16;
  cudaEvent_t e0, e1; cudaEventCreate(&e0); cudaEventCreate(&e1);
  int grids[] = {nsm * 4, nsm * 8, nsm * 16, nsm * 32};
  printf("\"copy_gbs\": {");
  for (int g = 0; g < 4; ++g) {
    float best = 1e30f;
    for (int r = 0; r < 6; ++r) {
      cudaEventRecord(e0); copy_v4<<<grids[g], 256>>>(a, b, n); cudaEventRecord(e1);
      CK(cudaEventSynchronize(e1)); float ms; cudaEventElapsedTime(&ms, e0, e1); if (ms < best) best = ms;
    }
    printf("%s\"g%d\": %.1f", g ? ", " : "", grids[g], 2.0 * bytes / (best * 1e-3) / 1e9);
  }
  printf("}, \"rmw_gbs\": {");
  for (int g = 0; g < 4; ++g) {
    float best = 1e30f;
    for (int r = 0; r < 6; ++r) {
      cudaEventRecord(e0); rmw_v4<<<grids[g], 256>>>(a, n); cudaEventRecord(e1);
      CK(cudaEventSynchronize(e1)); float ms; cudaEventElapsedTime(&ms, e0, e1); if (ms < best) best = ms;
    }
    printf("%s\"g%d\": %.1f", g ? ", " : "", grids[g], 2.0 * bytes / (best * 1e-3) / 1e9);
  }
  printf("}}\n");
  return 0;
}
