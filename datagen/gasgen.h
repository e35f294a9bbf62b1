/*
 * gasgen.h — seeded synthetic input generator (device side).
 *
 * Shared by the tests, the bench and smoke() as the ONE module that both the
 * CUDA path and the CPU oracle take their inputs from. It holds none of the
 * sort's arithmetic: it only produces float32 bit patterns from a counter
 * hash. The numpy twin is datagen/__init__.py; both implement exactly the
 *  recipe below, bit for bit (checked by
 * tests/test_gpu_parity.py::test_device_generator_matches_numpy).
 *
 * Recipe:
 *   mix(z)  = splitmix64 finalizer:
 *             z ^= z>>30; z *= 0xBF58476D1CE4E5B9; z ^= z>>27;
 *             z *= 0x94D049BB133111EB; z ^= z>>31            (mod 2^64)
 *   h(s,i,j)= mix( mix(s ^ ((i+1)*G)) + (j+1)*G ),  G = 0x9E3779B97F4A7C15
 *   hi = h>>32, lo = h & 0xFFFFFFFF.
 *   Distributions (value bits of element j of array i):
 *     0 paper_uniform  float32_rn(hi>>1): uniform integer in [0, 2^31-1]
 *                      stored as float
 *     1 uniform_bits   hi: every binary32 bit pattern (NaNs, -0, inf, ...)
 *     2 spectra_intensity ((127+popcount(lo&0xFFFF))<<23) | (hi>>9)
 *     3 spectra_mz     100 + float32(hi>>8) * (1900*2^-24)   (RN, no FMA)
 *     4 dup16          float32(hi>>28): 16 distinct values
 *     5 sorted         float32(b + j),       b = h(s,i,0xFFFFFFFF)>>41
 *     6 reverse        float32(b + n-1-j)
 *     7 special_mix    by lo % 1000: [0,100) -0; [100,200) +0; [200,225) +inf;
 *                      [225,250) -inf; [250,300) NaN (sign hi>>31, quiet bit
 *                      hi>>30&1, payload (hi&0x3FFFFF)|1); [300,320) subnormal
 *                      (sign hi>>31, fraction (hi&0x7FFFFF)|1); else
 *                      float32_rn((int32)hi) * (1000*2^-31)
 *   Array lengths of the ragged batch: len_i = lo + h(s^LEN_SALT, i, 0).hi % (hi-lo+1).
 */
#ifndef GASGEN_H
#define GASGEN_H
#include <stdint.h>
#include <cuda_runtime.h>
#ifdef __cplusplus
extern "C" {
#endif

/* d[(i-i0)*n + j] = value(dist, seed, i, j, n) for i in [i0, i0+N), j < n. Returns cudaError_t. */
int gasgen_fixed(uint32_t* d, int dist, uint64_t seed, int64_t i0, int64_t N, int32_t n,
                 cudaStream_t stream);
/* d[off[k] - off[0] + j] = value(dist, seed, i0+k, j, off[k+1]-off[k]) for k < N. */
int gasgen_ragged(uint32_t* d, const int64_t* d_off, int dist, uint64_t seed, int64_t i0,
                  int64_t N, cudaStream_t stream);

#ifdef __cplusplus
}
#endif
#endif
