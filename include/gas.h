/*
 * gas.h — C ABI of the B200-native GPU-ArraySort hot path (libgas.so).
 *
 * The operation (PAPER.md, cited "P:Lx-y" = line of the paper text):
 *   Definition 1 (§4): given a batch I of N unsorted arrays
 *   A_1..A_N of n elements, produce I' where every A'_i is A_i arranged as
 *   a1 <= a2 <= ... <= an. Arrays are independent,
 *   the result overwrites the input ("in-place", Abstract
 *   P:L38-39) and the elements are float32 (§7.2). The paper
 *   bounds the arrays it designs for at ~4000 elements (spectra peaks,
 *   P:L170-173), hence gas_max_array_len().
 *
 * Ordering (reading C-1): "<=" is IEEE 754-2008 §5.10 totalOrder:
 *   -NaN(quiet, larger payload first) < -NaN(signaling) < -inf < ... < -0
 *   < +0 < ... < +inf < +sNaN < +qNaN. The result of each array is a
 *   permutation of its input BIT PATTERNS (no float arithmetic is applied,
 *   so no NaN is quieted, no subnormal flushed). The output is unique, so
 *   every correct implementation is bit-identical (reading C-2).
 *
 * Conventions for every entry point:
 *   - Pointers named d_* are DEVICE memory of the current device, owned by
 *     the caller; the library never calls cudaSetDevice. Workspace, where an
 *     entry point needs any, is stream-ordered (allocated and freed on
 *     `stream`) from a library-owned memory pool per device that keeps its
 *     memory, so steady-state calls never allocate from the driver and never
 *     synchronise: gas_sort_arrays with 512 < array_len <= 1024 and
 *     num_arrays >= 16384, 4 * num_arrays + 4112 bytes (control block, the
 *     4 KB batch-CDF table, an array list); with array_len > 16384,
 *     4 * num_arrays + 8 bytes (n <= 32768) or that plus 64 * num_arrays + 8
 *     bytes of part offsets and the offsets sort's 72 bytes (n > 32768);
 *     gas_sort_pairs with 512 < array_len <= 1024, 4 * num_arrays + 4 bytes;
 *     gas_sort_arrays_offsets with max_array_len > 256, 72 bytes. Everything
 *     else: zero workspace.
 *   - Work is enqueued on `stream` (0 = legacy default stream) and the call
 *     returns without a host synchronisation. Argument and launch-
 *     configuration errors are returned synchronously; faults during
 *     execution surface at the caller's next synchronisation, as usual in
 *     CUDA.
 *   - All counts and element offsets are 64-bit; a batch may hold more than
 *     2^31 elements (e.g. 10^7 x 1000).
 *   - Functions are reentrant and thread-safe; concurrent calls on
 *     overlapping memory are the caller's race.
 *   - The device-resident entry points enqueue only kernels (and, for the
 *     offsets variant, one memset) on `stream`: after one warm-up call on a
 *     stream they can be captured into a CUDA graph and replayed
 *     (tests/test_gpu_parity.py::test_cuda_graph_capture_and_replay).
 *   - No C++ exceptions cross this boundary.
 */
#ifndef GAS_H
#define GAS_H

#include <stdint.h>
#include <cuda_runtime_api.h>

#ifdef __cplusplus
extern "C" {
#endif

/* Exported symbols of libgas.so (built with -fvisibility=hidden: kernels and
   helpers stay private, so a process can load several CUDA libraries that
   share kernel names without interposition). */
#if defined(__GNUC__)
#define GAS_API __attribute__((visibility("default")))
#else
#define GAS_API
#endif

typedef enum gas_status {
  GAS_SUCCESS = 0,
  GAS_ERROR_INVALID_VALUE = 1, /* NULL pointer with work to do; negative count/length;
                                  pointer not 4-byte aligned; bad offsets (GAS_CHECK=1) */
  GAS_ERROR_UNSUPPORTED = 2,   /* an array longer than gas_max_array_len() */
  GAS_ERROR_CUDA = 3           /* a CUDA call failed; raw cudaError_t in gas_last_cuda_error() */
} gas_status;

/*
 * Fixed-length batch (Definition 1): array i occupies
 * d_data[i*array_len .. (i+1)*array_len), i in [0, num_arrays); every array is
 * sorted ascending in place.
 *   d_data      device pointer, 4-byte aligned (16-byte aligned with
 *               array_len % 4 == 0 selects 128-bit vector loads/stores).
 *   num_arrays  N >= 0. array_len n >= 0. N == 0 or n <= 1: no-op, d_data may be NULL.
 *   n > gas_max_array_len(): GAS_ERROR_UNSUPPORTED, nothing enqueued.
 * One kernel launch per call, except 512 < n <= 1024 with N >= 16384
 * (BASELINE.json configs[1]-[4]): a device-routed pipeline of six launches
 * (four with rows that are not 16-byte aligned): a sampler kernel picks, on
 * the device, which kernel sorts the batch — value buckets, key-linear
 * buckets, batch-CDF buckets, the counting sort or the split kernel (special
 * values and equal-key runs); the others exit at once (csrc/sort1024.cuh);
 * its workspace is above. 16384 < n <= 65536: two launches (a thread-block
 * cluster kernel and the fallback for oversize parts), or, for n > 32768, the
 * partition kernel followed by the variable-length sort's launches.
 */
GAS_API gas_status gas_sort_arrays(float* d_data, int64_t num_arrays, int32_t array_len, cudaStream_t stream);

/*
 * Variable-length batch (BASELINE.json north_star "variable-length offsets
 * variant"; reading C-16): array i is d_data[d_offsets[i] ..
 * d_offsets[i+1]), d_offsets is int64[num_arrays+1] in DEVICE memory,
 * nondecreasing, d_offsets[0] >= 0. Arrays may be empty, adjacent and at any
 * 4-byte alignment; no byte outside [d_offsets[0], d_offsets[N]) is touched
 * and no array's bytes are written by another array's work.
 *   max_array_len  an upper bound on every length (0 = gas_max_array_len());
 *                  used to skip size classes that cannot occur. A length above
 *                  it is undefined behaviour unless the environment variable
 *                  GAS_CHECK=1 is set, in which case the offsets are validated
 *                  on the device first (with a stream synchronisation) and a
 *                  violation returns GAS_ERROR_INVALID_VALUE with nothing sorted.
 *   max_array_len > gas_max_array_len(): GAS_ERROR_UNSUPPORTED.
 * Workspace: 72 bytes per call for dynamic scheduling when max_array_len >
 * 256 (stream-ordered, from the library's pool; each call and each captured
 * graph has its own).
 * One kernel launch per size class up to max_array_len (at most 17 launches:
 * powers of two up to 2048, then (2048,3072], (3072,4096], (4096,6144],
 * (6144,8192], (8192,12288], (12288,16384]). The launches are forked over 8
 * library-owned non-blocking streams per (device, stream) (created on first
 * use, with their fork/join events) and joined back into `stream` before the
 * call returns, so work enqueued later on `stream` still runs after the sort
 * and the call can be captured into a CUDA graph. GAS_OFFSETS_STREAMS=k
 * (1..8) sets the fan-out; 1 keeps every launch on `stream`. At most 64 caller
 * streams per process get such a set; calls on further streams launch on
 * `stream` alone. gas_release_stream() frees a stream's set.
 */
GAS_API gas_status gas_sort_arrays_offsets(float* d_data, const int64_t* d_offsets, int64_t num_arrays,
                                   int32_t max_array_len, cudaStream_t stream);

/*
 * Key + payload variant (north_star "optional key+payload variant"; SURVEY.md
 * §8(f) row f2): keys as in gas_sort_arrays, d_values[i*n + j] is carried with
 * d_keys[i*n + j]. STABLE: equal keys (identical bit patterns) keep their input
 * order, so the payload order is unique (reading C-2). Same argument rules as
 * gas_sort_arrays (both pointers 4-byte aligned), except that array_len is
 * limited to 8192 (GAS_ERROR_UNSUPPORTED above).
 */
GAS_API gas_status gas_sort_pairs(float* d_keys, uint32_t* d_values, int64_t num_arrays, int32_t array_len,
                          cudaStream_t stream);

/*
 * Host-memory convenience entry point (the paper's
 * future-work out-of-core sort): h_data is HOST memory holding
 * the fixed-length batch; it is streamed through the current device in
 * chunks (host->device copy, sort, device->host copy on rotating streams so
 * the two copy directions and the sort overlap) and the sorted batch is
 * written back to h_data. Pinned (page-locked) host memory gives full-duplex
 * PCIe; pageable memory works but is much slower (measured for 2M x 1000 on
 * one B200: 175 ms pinned, 1.14 s pageable — register or pin the buffer). BLOCKING: returns after the
 * result is in h_data. Device staging (3 x 128 MB by default, GAS_HOST_CHUNK_MB /
 * GAS_HOST_SLOTS) and its streams are allocated on first use per device and kept
 * for later calls; concurrent host-path calls on one device are serialised.
 */
GAS_API gas_status gas_sort_arrays_host(float* h_data, int64_t num_arrays, int32_t array_len);

/*
 * Host-memory variant of gas_sort_arrays_offsets (SURVEY.md §8(f) row f1 for
 * ragged batches, the out-of-core spectra batches of P:L573-584): h_data and
 * h_offsets are HOST memory (CSR as in gas_sort_arrays_offsets). The batch is
 * cut at array boundaries into chunks of at most 128 MB (GAS_HOST_CHUNK_MB)
 * and 2^20 arrays, streamed through the current device with the same
 * overlapped H2D / sort / D2H as gas_sort_arrays_host, and written back in
 * place. BLOCKING. Same argument rules as gas_sort_arrays_offsets; bytes
 * outside [h_offsets[0], h_offsets[N]) are never read or written. Staging
 * (data, pinned and device offsets buffers) is kept per device for later calls.
 */
GAS_API gas_status gas_sort_arrays_offsets_host(float* h_data, const int64_t* h_offsets, int64_t num_arrays,
                                                int32_t max_array_len);

/* Releases the side streams and events gas_sort_arrays_offsets created for
   (current device, stream), after the work already enqueued on them has
   finished (host-blocking on those streams only). Call it before destroying a
   stream that was used with the offsets variant; a no-op for other streams. */
GAS_API gas_status gas_release_stream(cudaStream_t stream);

/* Largest supported array length of gas_sort_arrays / _offsets / _host: 16384,
   4x the paper's spectra bound of ~4000 peaks. */
GAS_API int32_t gas_max_array_len(void);

/* Static, human-readable name of a status code. */
GAS_API const char* gas_status_string(gas_status s);

/* cudaError_t of the most recent GAS_ERROR_CUDA on this host thread (0 if none). */
GAS_API int gas_last_cuda_error(void);

/* Number of kernels this library has launched in this process (monotone counter;
   bench.py reports the delta over its timed region as "gpu_launches"). */
GAS_API int64_t gas_launch_count(void);

#ifdef __cplusplus
}
#endif
#endif /* GAS_H */
