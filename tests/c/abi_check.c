/* Plain-C client of include/gas.h: proves the boundary is a C ABI (no C++,
 * no torch) and exercises the host-side validation paths, which return before
 * any CUDA call (so this runs on a machine without a GPU). With a GPU and
 * argv[1] == "gpu" it also sorts a small batch through host memory and checks
 * the result is nondecreasing in IEEE totalOrder. */
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>
#include <string.h>

#include "gas.h"

static int fails = 0;
#define CHECK(cond) do { if (!(cond)) { fprintf(stderr, "FAIL %s:%d %s\n", __FILE__, __LINE__, #cond); ++fails; } } while (0)

static uint32_t key(uint32_t u) { return u ^ ((u >> 31) ? 0xFFFFFFFFu : 0x80000000u); }

int main(int argc, char** argv) {
  CHECK(gas_max_array_len() == 65536);
  CHECK(strcmp(gas_status_string(GAS_SUCCESS), "GAS_SUCCESS") == 0);
  CHECK(gas_sort_arrays(NULL, 0, 1000, 0) == GAS_SUCCESS);
  CHECK(gas_sort_arrays(NULL, 5, 1, 0) == GAS_SUCCESS);
  CHECK(gas_sort_arrays(NULL, -1, 10, 0) == GAS_ERROR_INVALID_VALUE);
  CHECK(gas_sort_arrays(NULL, 10, 10, 0) == GAS_ERROR_INVALID_VALUE);
  CHECK(gas_sort_arrays((float*)(uintptr_t)0x1000, 10, 65537, 0) == GAS_ERROR_UNSUPPORTED);
  CHECK(gas_sort_arrays_offsets((float*)(uintptr_t)0x1000, (const int64_t*)(uintptr_t)0x2000, 10, 16385, 0) == GAS_ERROR_UNSUPPORTED);
  CHECK(gas_sort_pairs((float*)(uintptr_t)0x1000, (uint32_t*)(uintptr_t)0x2000, 10, 8193, 0) == GAS_ERROR_UNSUPPORTED);
  CHECK(gas_sort_arrays_offsets(NULL, NULL, 0, 0, 0) == GAS_SUCCESS);
  CHECK(gas_sort_arrays_host(NULL, 3, 10) == GAS_ERROR_INVALID_VALUE);
  CHECK(gas_launch_count() == 0);
  if (argc > 1 && strcmp(argv[1], "gpu") == 0) {
    const int64_t N = 1000; const int32_t n = 1000;
    uint32_t* h = (uint32_t*)malloc(sizeof(uint32_t) * N * n);
    uint64_t x = 0x20160815ull;
    for (int64_t i = 0; i < N * n; ++i) { x = x * 6364136223846793005ull + 1442695040888963407ull; h[i] = (uint32_t)(x >> 32); }
    CHECK(gas_sort_arrays_host((float*)h, N, n) == GAS_SUCCESS);
    for (int64_t i = 0; i < N; ++i)
      for (int32_t j = 1; j < n; ++j) CHECK(key(h[i * n + j - 1]) <= key(h[i * n + j]));
    CHECK(gas_launch_count() >= 1);
    free(h);
  }
  if (fails == 0) printf("abi_check OK\n");
  return fails ? 1 : 0;
}
