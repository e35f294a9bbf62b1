// Experiment harness for the counting-sort/window kernel (csrc/cw1024.cuh):
// per distribution, times k_fixed_cw1024 against gas_sort_arrays (libgas.so,
// itself parity-tested against the oracle) on the same seeded batch, checks
// the two outputs bit for bit on the device, and reports how many arrays took
// the network fallback. Usage: cw_exp [N=2000000] [n=1000] [steps=10] [dists=0,1,2,3,4,5,6,7]
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <vector>
#include <algorithm>
#include <cuda_runtime.h>
#include "gas.h"
#include "gasgen.h"
extern "C" int cw_info(int* regs, long long* local_bytes, int* grid_cap);
extern "C" int cw_launch(uint32_t* d, long long N, int n, unsigned long long* stats, cudaStream_t s);
extern "C" int s1_launch(uint32_t* d, long long N, int n, cudaStream_t s);

#define CK(x) do { cudaError_t e_ = (x); if (e_ != cudaSuccess) { std::fprintf(stderr, "%s:%d %s: %s\n", __FILE__, __LINE__, #x, cudaGetErrorString(e_)); std::exit(1); } } while (0)

__global__ void k_diff(const uint32_t* a, const uint32_t* b, size_t n, unsigned long long* cnt) {
  unsigned long long c = 0;
  for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n; i += (size_t)gridDim.x * blockDim.x) c += a[i] != b[i];
  if (c) atomicAdd(cnt, c);
}

static const char* kNames[] = {"paper_uniform", "uniform_bits", "spectra_intensity", "spectra_mz",
                               "dup16", "sorted", "reverse", "special_mix"};

int main(int argc, char** argv) {
  const long long N = argc > 1 ? std::atoll(argv[1]) : 2000000;
  const int n = argc > 2 ? std::atoi(argv[2]) : 1000;
  const int steps = argc > 3 ? std::atoi(argv[3]) : 10;
  std::vector<int> dists;
  {
    const char* s = argc > 4 ? argv[4] : "0,1,2,3,4,5,6,7";
    for (const char* p = s; *p;) { dists.push_back(std::atoi(p)); while (*p && *p != ',') ++p; if (*p) ++p; }
  }
  const size_t words = (size_t)N * n, bytes = words * 4;
  uint32_t *pristine, *work, *ref;
  unsigned long long *stats, *diff;
  CK(cudaMalloc(&pristine, bytes));
  CK(cudaMalloc(&work, bytes));
  CK(cudaMalloc(&ref, bytes));
  CK(cudaMalloc(&stats, 8));
  CK(cudaMalloc(&diff, 8));
  int regs = 0, cap = 0, sms = 0;
  long long lbytes = 0;
  if (cw_info(&regs, &lbytes, &cap) != 0) { std::fprintf(stderr, "cw_info failed\n"); return 1; }
  CK(cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0));
  std::printf("{\"kernel\": \"k_fixed_cw1024\", \"regs\": %d, \"local_bytes\": %lld, \"grid_cap\": %d}\n", regs, lbytes, cap);
  cudaEvent_t e0, e1;
  CK(cudaEventCreate(&e0));
  CK(cudaEventCreate(&e1));
  for (int dist : dists) {
    if (gasgen_fixed(pristine, dist, 0x20160815ull + 1, 0, N, n, 0) != 0) return 1;
    std::vector<float> tr, tc;
    for (int s = 0; s < steps + 2; ++s) {
      CK(cudaMemcpy(work, pristine, bytes, cudaMemcpyDeviceToDevice));
      CK(cudaEventRecord(e0));
      if (gas_sort_arrays(reinterpret_cast<float*>(work), N, n, 0) != GAS_SUCCESS) return 1;
      CK(cudaEventRecord(e1));
      CK(cudaEventSynchronize(e1));
      float t;
      CK(cudaEventElapsedTime(&t, e0, e1));
      if (s >= 2) tr.push_back(t);
    }
    CK(cudaMemcpy(ref, work, bytes, cudaMemcpyDeviceToDevice));
    unsigned long long fall = 0, nd = 0;
    for (int s = 0; s < steps + 2; ++s) {
      CK(cudaMemcpy(work, pristine, bytes, cudaMemcpyDeviceToDevice));
      CK(cudaMemset(stats, 0, 8));
      CK(cudaEventRecord(e0));
      if (cw_launch(work, N, n, s == 0 ? stats : nullptr, 0) != 0) { std::fprintf(stderr, "cw_launch failed\n"); return 1; }
      CK(cudaEventRecord(e1));
      CK(cudaEventSynchronize(e1));
      float t;
      CK(cudaEventElapsedTime(&t, e0, e1));
      if (s == 0) CK(cudaMemcpy(&fall, stats, 8, cudaMemcpyDeviceToHost));
      if (s >= 2) tc.push_back(t);
    }
    CK(cudaMemset(diff, 0, 8));
    k_diff<<<sms * 8, 256>>>(work, ref, words, diff);
    CK(cudaMemcpy(&nd, diff, 8, cudaMemcpyDeviceToHost));
    std::vector<float> ts;
    unsigned long long nd1 = 0;
    for (int s = 0; s < steps + 2; ++s) {
      CK(cudaMemcpy(work, pristine, bytes, cudaMemcpyDeviceToDevice));
      CK(cudaEventRecord(e0));
      if (s1_launch(work, N, n, 0) != 0) { std::fprintf(stderr, "s1_launch failed\n"); return 1; }
      CK(cudaEventRecord(e1));
      CK(cudaEventSynchronize(e1));
      float t;
      CK(cudaEventElapsedTime(&t, e0, e1));
      if (s >= 2) ts.push_back(t);
    }
    CK(cudaMemset(diff, 0, 8));
    k_diff<<<sms * 8, 256>>>(work, ref, words, diff);
    CK(cudaMemcpy(&nd1, diff, 8, cudaMemcpyDeviceToHost));
    std::sort(ts.begin(), ts.end());
    const double m1 = ts[ts.size() / 2];
    std::sort(tr.begin(), tr.end());
    std::sort(tc.begin(), tc.end());
    const double mr = tr[tr.size() / 2], mc = tc[tc.size() / 2];
    std::printf("{\"dist\": \"%s\", \"N\": %lld, \"n\": %d, \"ref_ms\": %.4f, \"cw_ms\": %.4f, \"cw_frac\": %.4f, "
                "\"ref_frac\": %.4f, \"fallback_arrays\": %llu, \"mismatched_words\": %llu, \"s1_ms\": %.4f, \"s1_frac\": %.4f, \"s1_mismatched\": %llu}\n",
                kNames[dist], N, n, mr, mc, 2.0 * bytes / (mc * 1e-3) / 6544e9, 2.0 * bytes / (mr * 1e-3) / 6544e9,
                fall, nd, m1, 2.0 * bytes / (m1 * 1e-3) / 6544e9, nd1);
    std::fflush(stdout);
  }
  return 0;
}
