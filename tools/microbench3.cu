// FP64 min/max (DMNMX) throughput on sm_100a, alone and co-issued with VIMNMX / IMAD:
// can the FP64 pipe carry part of a compare-exchange network? Keys as doubles 2^52 + k.
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>
constexpr int ITERS = 2048;
__device__ __forceinline__ double mkd(uint32_t k) { return __hiloint2double(0x43300000, (int)k); }
__global__ void __launch_bounds__(1024) k_dmnmx(double* out, unsigned long long* cyc, uint32_t seed) {
  double x[8], y[8];
  for (int c = 0; c < 8; ++c) { x[c] = mkd(seed * (threadIdx.x + 1) + c); y[c] = mkd(seed ^ (c * 977u + threadIdx.x)); }
  __syncthreads(); unsigned long long t0 = clock64();
  for (int it = 0; it < ITERS; ++it) {
#pragma unroll
    for (int c = 0; c < 8; ++c) { double a = x[c], b = y[c]; x[c] = fmin(a, b); y[c] = fmax(a, b) + 0.0; }
  }
  __syncthreads(); unsigned long long t1 = clock64();
  double acc = 0; for (int c = 0; c < 8; ++c) acc += x[c] + y[c];
  out[blockIdx.x * blockDim.x + threadIdx.x] = acc; if (threadIdx.x == 0) cyc[blockIdx.x] = t1 - t0;
}
// mixed: per CE one VIMNMX (min) on lo words + one DMNMX (max) on doubles
__global__ void __launch_bounds__(1024) k_mixed(double* out, unsigned long long* cyc, uint32_t seed) {
  double x[8], y[8];
  for (int c = 0; c < 8; ++c) { x[c] = mkd(seed * (threadIdx.x + 1) + c); y[c] = mkd(seed ^ (c * 977u + threadIdx.x)); }
  __syncthreads(); unsigned long long t0 = clock64();
  for (int it = 0; it < ITERS; ++it) {
#pragma unroll
    for (int c = 0; c < 8; ++c) {
      double a = x[c], b = y[c];
      uint32_t mn = min((uint32_t)__double2loint(a), (uint32_t)__double2loint(b));
      y[c] = fmax(a, b);
      x[c] = __hiloint2double(0x43300000, (int)mn);
    }
  }
  __syncthreads(); unsigned long long t1 = clock64();
  double acc = 0; for (int c = 0; c < 8; ++c) acc += x[c] + y[c];
  out[blockIdx.x * blockDim.x + threadIdx.x] = acc; if (threadIdx.x == 0) cyc[blockIdx.x] = t1 - t0;
}
typedef void (*F)(double*, unsigned long long*, uint32_t);
int main() {
  int nsm; cudaDeviceGetAttribute(&nsm, cudaDevAttrMultiProcessorCount, 0);
  double* out; unsigned long long* cyc; cudaMalloc(&out, nsm * 1024 * 8); cudaMalloc(&cyc, nsm * 8);
  struct { const char* n; F f; double ops; } ks[] = {{"dmnmx_pairs", k_dmnmx, 2}, {"mixed_vimnmx_dmnmx_CE", k_mixed, 1}};
  printf("{");
  for (int q = 0; q < 2; ++q) {
    ks[q].f<<<nsm, 1024>>>(out, cyc, 3u); cudaDeviceSynchronize();
    ks[q].f<<<nsm, 1024>>>(out, cyc, 12345u); cudaDeviceSynchronize();
    unsigned long long h[1024]; cudaMemcpy(h, cyc, nsm * 8, cudaMemcpyDeviceToHost);
    double mx = 0; for (int i = 0; i < nsm; ++i) mx = h[i] > mx ? h[i] : mx;
    printf("%s\"%s_per_clk_per_sm\": %.2f", q ? ", " : "", ks[q].n, 1024.0 * ITERS * 8 * ks[q].ops / mx);
  }
  printf(", \"err\": \"%s\"}\n", cudaGetErrorString(cudaGetLastError()));
}
