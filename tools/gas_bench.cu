// C++-only benchmark of the C ABI (no Python, no torch): generates the
// configs[1] batch on the device with the seeded generator, then times
// gas_sort_arrays with CUDA events (pristine copy restored before each step,
// untimed). Usage: gas_bench [num_arrays=2000000] [array_len=1000] [steps=20]
#include <cstdio>
#include <cstdlib>
#include <vector>
#include <algorithm>
#include <cuda_runtime.h>
#include "gas.h"
#include "gasgen.h"

#define CK(x) do { cudaError_t e_ = (x); if (e_ != cudaSuccess) { std::fprintf(stderr, "%s: %s\n", #x, cudaGetErrorString(e_)); return 1; } } while (0)

int main(int argc, char** argv) {
  const long long N = argc > 1 ? std::atoll(argv[1]) : 2000000;
  const int n = argc > 2 ? std::atoi(argv[2]) : 1000;
  const int steps = argc > 3 ? std::atoi(argv[3]) : 20;
  const size_t bytes = (size_t)N * n * 4;
  uint32_t *pristine = nullptr, *work = nullptr;
  CK(cudaMalloc(&pristine, bytes));
  CK(cudaMalloc(&work, bytes));
  if (gasgen_fixed(pristine, 0, 0x20160815ull + 1, 0, N, n, 0) != 0) return 1;
  cudaEvent_t a, b;
  CK(cudaEventCreate(&a));
  CK(cudaEventCreate(&b));
  std::vector<float> ms;
  for (int s = 0; s < steps + 3; ++s) {
    CK(cudaMemcpy(work, pristine, bytes, cudaMemcpyDeviceToDevice));
    CK(cudaEventRecord(a));
    const gas_status st = gas_sort_arrays(reinterpret_cast<float*>(work), N, n, 0);
    if (st != GAS_SUCCESS) { std::fprintf(stderr, "gas_sort_arrays: %s\n", gas_status_string(st)); return 1; }
    CK(cudaEventRecord(b));
    CK(cudaEventSynchronize(b));
    float t = 0;
    CK(cudaEventElapsedTime(&t, a, b));
    if (s >= 3) ms.push_back(t);
  }
  std::sort(ms.begin(), ms.end());
  const double med = ms[ms.size() / 2];
  std::printf("{\"num_arrays\": %lld, \"array_len\": %d, \"median_ms\": %.4f, \"min_ms\": %.4f, "
              "\"arrays_per_s\": %.4g, \"algorithmic_GBps\": %.1f}\n",
              N, n, med, ms.front(), N / (med * 1e-3), 2.0 * bytes / (med * 1e-3) / 1e9);
  return 0;
}
