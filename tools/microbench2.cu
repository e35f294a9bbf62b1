// Throughput of warp-level ranking primitives on sm_100a (radix-sort feasibility):
// MATCH.ANY, POPC, BREV/FLO, VOTE, ATOMS (distinct and colliding), REDUX.
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>
constexpr int ITERS = 2048;
#define K(NAME, ...) __global__ void __launch_bounds__(1024) NAME(uint32_t* out, unsigned long long* cyc, uint32_t seed) { \
  __shared__ uint32_t sh[8192]; for (int i = threadIdx.x; i < 8192; i += blockDim.x) sh[i] = 0; __syncthreads(); \
  uint32_t x[8]; for (int c = 0; c < 8; ++c) x[c] = (seed * (threadIdx.x + 7) + c * 2654435761u) >> (c & 7); \
  uint32_t acc = 0; unsigned long long t0 = clock64(); \
  for (int it = 0; it < ITERS; ++it) { _Pragma("unroll") for (int c = 0; c < 8; ++c) { __VA_ARGS__; } } \
  __syncthreads(); unsigned long long t1 = clock64(); \
  out[blockIdx.x * blockDim.x + threadIdx.x] = acc + x[0] + x[7] + sh[threadIdx.x]; if (threadIdx.x == 0) cyc[blockIdx.x] = t1 - t0; }
K(k_match, { uint32_t m = __match_any_sync(0xffffffffu, x[c] & 255u); acc += m; x[c] = x[c] * 1664525u + m; })
K(k_popc, { acc += __popc(x[c]); x[c] = x[c] * 1664525u + acc; })
K(k_ballot, { uint32_t b = __ballot_sync(0xffffffffu, x[c] & 1u); acc += b; x[c] = (x[c] >> 1) + b; })
K(k_atoms_distinct, { uint32_t r = atomicAdd(&sh[(threadIdx.x * 8 + c) & 8191], 1u); acc += r; x[c] += r; })
K(k_atoms_rand, { uint32_t r = atomicAdd(&sh[(x[c] & 255u) + (threadIdx.x >> 5) * 256], 1u); acc += r; x[c] = x[c] * 1664525u + r; })
K(k_redg, { atomicAdd(&sh[(x[c] & 255u) + (threadIdx.x >> 5) * 256], 1u); x[c] = x[c] * 1664525u + 1013904223u; })
K(k_sts_rand, { sh[(x[c] >> 3) & 8191] = x[c]; x[c] = x[c] * 1664525u + 1013904223u; })
K(k_lds_rand, { uint32_t v = sh[(x[c] >> 3) & 8191]; acc += v; x[c] = x[c] * 1664525u + 1013904223u + v; })
typedef void (*F)(uint32_t*, unsigned long long*, uint32_t);
int main() {
  int nsm; cudaDeviceGetAttribute(&nsm, cudaDevAttrMultiProcessorCount, 0);
  uint32_t* out; unsigned long long* cyc; cudaMalloc(&out, nsm * 1024 * 4); cudaMalloc(&cyc, nsm * 8);
  struct { const char* n; F f; } ks[] = {{"match_any", k_match}, {"popc", k_popc}, {"ballot", k_ballot},
    {"atoms_distinct", k_atoms_distinct}, {"atoms_rand256_per_warp", k_atoms_rand}, {"red_shared_rand", k_redg},
    {"sts_random", k_sts_rand}, {"lds_random", k_lds_rand}};
  printf("{\"lane_ops_per_clk_per_sm\": {");
  for (size_t q = 0; q < sizeof(ks) / sizeof(ks[0]); ++q) {
    ks[q].f<<<nsm, 1024>>>(out, cyc, 1u); cudaDeviceSynchronize();
    ks[q].f<<<nsm, 1024>>>(out, cyc, 12345u); cudaDeviceSynchronize();
    unsigned long long h[1024]; cudaMemcpy(h, cyc, nsm * 8, cudaMemcpyDeviceToHost);
    double mx = 0; for (int i = 0; i < nsm; ++i) mx = h[i] > mx ? h[i] : mx;
    printf("%s\"%s\": %.2f", q ? ", " : "", ks[q].n, 1024.0 * ITERS * 8 / mx);
  }
  printf("}, \"err\": \"%s\"}\n", cudaGetErrorString(cudaGetLastError()));
}
