// bucket_cta.cuh — the bucket-then-network sort of bucket1024.cuh for one
// array per CTA of W = 1, 2 or 4 warps (n <= 1024 W keys, 32 per thread):
// the fixed-length classes 1024 < n <= 4096, unaligned rows with
// 512 < n <= 1024, and the variable-length (CSR offsets) classes
// 512 < len <= 4096 of BASELINE.json configs[3] (spectra).
//
// Same method and correctness argument as bucket1024.cuh (value buckets from
// one monotone FADD + FFMA map, ranks from shared atomics, <= 32 keys per
// bucket sorted by a 32-key register network, warp-uniform fallback to the
// whole-array network), with 62 W buckets so that a bucket still holds ~16
// keys; thread t sorts buckets t and t + 32 W. CTA-wide steps (min/max,
// bucket bases, the fallback vote) go through shared memory and barriers.
#pragma once
#include <cstdint>

#include "bucket1024.cuh"
#include "segsort.cuh"
#include "warp1024.cuh"

namespace gas {

template <int W>
struct BkCta {
  static constexpr int T = 32 * W;         // threads
  static constexpr int P = 1024 * W;       // capacity (keys)
  static constexpr int NB = 62 * W;        // buckets 0 .. NB-1
  static constexpr int ROWS = 64 * W;      // bucket rows (the last 2 W stay empty)
  static constexpr int CNT_BYTES = ROWS * 4;
  static constexpr int SLOT_BYTES = ROWS * kBkRowWords * 4;
  static constexpr int RED_BYTES = 16 * 4;  // cross-warp min/max and scan partials
  static constexpr int SMEM = CNT_BYTES + SLOT_BYTES + RED_BYTES;
  // the fallback network needs P words of exchange + 4 KB per warp
  static_assert(P * 4 + W * 4096 <= SLOT_BYTES, "fallback scratch fits in the slot buffer");
};

#ifndef GAS_BKC_WARPS_PER_SM
#define GAS_BKC_WARPS_PER_SM 16
#endif

// Sort the n keys at `arr` (P/2 < n <= P; VEC: 16-byte-aligned, n % 4 == 0)
// in place. All T threads of the CTA call it; `sm` is BkCta<W>::SMEM bytes.
template <int W, bool VEC>
__device__ __forceinline__ void bucket_sort_cta(uint32_t* __restrict__ arr, int n, unsigned char* sm, uint32_t one) {
  using C = BkCta<W>;
  constexpr int T = C::T;
  const int t = threadIdx.x, lane = t & 31, warp = t >> 5;
  const uint32_t cnt_sa = (uint32_t)__cvta_generic_to_shared(sm);
  const uint32_t slot_sa = cnt_sa + C::CNT_BYTES;
  unsigned char* const slot_ptr = sm + C::CNT_BYTES;
  float* const red = reinterpret_cast<float*>(sm + C::CNT_BYTES + C::SLOT_BYTES);
  const uint32_t cnt_b0 = cnt_sa - 0x4B000000u * 4u;
  const uint32_t slot_c0 = slot_sa - (uint32_t)kBkRowWords * cnt_sa;
  const int nc = n >> 2;
  // key r of this thread: VEC element 4 (t + T (r/4)) + r%4, else element t + T r
  auto valid = [&](int r) -> bool {
    if (VEC) return (r >> 2) < 4 || t + T * (r >> 2) < nc;
    return r < 16 || t + T * r < n;
  };

  // ---- stage in (raw bits); slots past the end stay out of every step
  uint32_t k[32];
  if constexpr (VEC) {
    const uint4* src = reinterpret_cast<const uint4*>(arr);
#pragma unroll
    for (int q = 0; q < 8; ++q) {
      uint4 v = make_uint4(0, 0, 0, 0);
      if (valid(4 * q)) v = ld_stream(src + t + T * q);
      k[4 * q] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
    }
  } else {
#pragma unroll
    for (int r = 0; r < 32; ++r) k[r] = valid(r) ? ld_stream(arr + t + T * r) : 0u;
  }
  // ---- min / max over the valid keys (NaN-propagating), then across the CTA
  float vmin = __uint_as_float(k[0]), vmax = vmin;
#pragma unroll
  for (int r = 1; r < 16; ++r) {
    vmin = fmin_nan(vmin, __uint_as_float(k[r]));
    vmax = fmax_nan(vmax, __uint_as_float(k[r]));
  }
#pragma unroll
  for (int r = 16; r < 32; ++r)
    if (valid(r)) {
      vmin = fmin_nan(vmin, __uint_as_float(k[r]));
      vmax = fmax_nan(vmax, __uint_as_float(k[r]));
    }
#pragma unroll
  for (int m = 16; m >= 1; m >>= 1) {
    vmin = fmin_nan(vmin, __shfl_xor_sync(0xffffffffu, vmin, m));
    vmax = fmax_nan(vmax, __shfl_xor_sync(0xffffffffu, vmax, m));
  }
  if constexpr (W > 1) {
    if (lane == 0) { red[2 * warp] = vmin; red[2 * warp + 1] = vmax; }
    __syncthreads();
#pragma unroll
    for (int w = 0; w < W; ++w) {
      vmin = fmin_nan(vmin, red[2 * w]);
      vmax = fmax_nan(vmax, red[2 * w + 1]);
    }
  }
  const float range = __fsub_rn(vmax, vmin);
  const float s = __fdiv_rn((float)(C::NB - 1), range);
  bool use_buckets = fabsf(vmin) <= 3.402823466e38f && fabsf(vmax) <= 3.402823466e38f && range > 0.0f &&
                     range <= 3.402823466e38f && s <= 3.402823466e38f;
  const bool raw = vmin > 0.0f;
  uint32_t t0 = 0, t1 = 0, base0 = 0, base1 = 0;
  if (use_buckets) {  // CTA-uniform
#pragma unroll
    for (int q = 0; q < C::SLOT_BYTES / 16 / T; ++q)
      sts128(slot_sa + (t + T * q) * 16, make_uint4(kPadKey, kPadKey, kPadKey, kPadKey));
    if (t < C::ROWS / 4) sts128(cnt_sa + t * 16, make_uint4(0, 0, 0, 0));
    __syncthreads();
    uint32_t rk[32];
#pragma unroll
    for (int r = 0; r < 32; ++r) rk[r] = atoms_inc_if(valid(r), bucket_bits(k[r], vmin, s) * 4u + cnt_b0);
    __syncthreads();
    t0 = lds32(cnt_sa + t * 4);
    t1 = lds32(cnt_sa + (T + t) * 4);
    use_buckets = __syncthreads_and(t0 <= 32u && t1 <= 32u);
    if (use_buckets) {
      // bucket bases: exclusive scan of the 2T bucket sizes (two 16-bit halves)
      uint32_t x = t0 | (t1 << 16);
#pragma unroll
      for (int m = 1; m < 32; m <<= 1) {
        const uint32_t y = __shfl_up_sync(0xffffffffu, x, m);
        if (lane >= m) x += y;
      }
      uint32_t before = 0, total = __shfl_sync(0xffffffffu, x, 31);
      if constexpr (W > 1) {
        uint32_t* const part = reinterpret_cast<uint32_t*>(red) + 8;
        if (lane == 31) part[warp] = x;
        __syncthreads();
        total = 0;
#pragma unroll
        for (int w = 0; w < W; ++w) {
          const uint32_t pw = part[w];
          before += (w < warp) ? pw : 0u;
          total += pw;
        }
      }
      x += before;
      base0 = (x & 0xFFFFu) - t0;
      base1 = (total & 0xFFFFu) + (x >> 16) - t1;
#pragma unroll
      for (int r = 0; r < 32; ++r) {
        const uint32_t ca = bucket_bits(k[r], vmin, s) * 4u + cnt_b0;
        sts32_if(valid(r), ca * (uint32_t)kBkRowWords + (rk[r] * 4u + slot_c0), raw ? k[r] : key_from_bits(k[r]));
      }
      __syncthreads();
    }
  }

  if (use_buckets) {
    // two rounds: bucket t, then bucket t + T; the output is staged at word p
    // of the slot buffer (rows 0 .. T-1 hold >= 36 T >= n words and are free
    // after round 0's gather; round 1 reads rows T .. 2T-1 only)
    const uint32_t out_sa = slot_sa;
#pragma unroll 1
    for (int rho = 0; rho < 2; ++rho) {
      const uint32_t row = slot_sa + (t + T * rho) * (kBkRowWords * 4);
#pragma unroll
      for (int q = 0; q < 8; ++q) {
        const uint4 v = lds128(row + q * 16);
        k[4 * q] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
      }
      __syncthreads();
      sort32_bk(k, one);
      const uint32_t tb = rho ? t1 : t0;
      const uint32_t ob = out_sa + (rho ? base1 : base0) * 4;
      if (raw) {
#pragma unroll
        for (int i = 0; i < 32; ++i) sts32_if((uint32_t)i < tb, ob + i * 4, k[i]);
      } else {
#pragma unroll
        for (int i = 0; i < 32; ++i) sts32_if((uint32_t)i < tb, ob + i * 4, bits_from_key(k[i]));
      }
    }
    __syncthreads();
    if constexpr (VEC) {
      uint4* dst = reinterpret_cast<uint4*>(arr);
#pragma unroll
      for (int q = 0; q < 8; ++q) {
        const int c = t + T * q;
        if (c < nc) st_stream(dst + c, lds128(out_sa + c * 16));
      }
    } else {
#pragma unroll
      for (int r = 0; r < 32; ++r) {
        const int e = t + T * r;
        if (e < n) st_stream(arr + e, lds32(out_sa + e * 4));
      }
    }
  } else {
    // ---- fallback: the whole-array network (warp1024.cuh sort_cta)
#pragma unroll
    for (int r = 0; r < 32; ++r) k[r] = valid(r) ? key_from_bits(k[r]) : kPadKey;
    uint32_t* xs = reinterpret_cast<uint32_t*>(slot_ptr);
    uint32_t* wbuf = xs + C::P + warp * 1024;
    __syncthreads();
    sort_cta<W>(k, t, lane, xs, wbuf, one);
    __syncthreads();
    uint4* sb = reinterpret_cast<uint4*>(slot_ptr);
    stage_out_words<32>(k, sb, t * 32);
    __syncthreads();
    if constexpr (VEC) {
#pragma unroll
      for (int q = 0; q < 8; ++q) {
        const int c = t + T * q;
        if (c < nc) st_stream(reinterpret_cast<uint4*>(arr) + c, sb[swz(c)]);
      }
    } else {
#pragma unroll
      for (int r = 0; r < 32; ++r) {
        const int e = t + T * r;
        if (e < n) st_stream(arr + e, sword(sb, e));
      }
    }
  }
  __syncthreads();  // the next array reuses the shared buffers
}

// Fixed length, one array per CTA (persistent grid-stride).
template <int W, bool VEC>
__global__ void __launch_bounds__(32 * W, GAS_BKC_WARPS_PER_SM / W)
    k_fixed_bucket_cta(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one) {
  extern __shared__ __align__(16) unsigned char bkc_smem[];
  for (int64_t a = blockIdx.x; a < N; a += gridDim.x) bucket_sort_cta<W, VEC>(d + a * (int64_t)n, n, bkc_smem, one);
}

// Variable length: the arrays with LO < len <= HI (P/2 <= LO, HI <= P), found
// by scanning windows of 32 arrays handed out dynamically through `ctr` (one
// counter per launch, zeroed by the host), as k_offsets_cta. Rows may start
// at any 4-byte boundary: scalar loads and stores.
template <int W>
__global__ void __launch_bounds__(32 * W, GAS_BKC_WARPS_PER_SM / W)
    k_offsets_bucket(uint32_t* __restrict__ d, const int64_t* __restrict__ off, int64_t N, int64_t LO, int64_t HI,
                     unsigned long long* __restrict__ ctr, uint32_t one) {
  extern __shared__ __align__(16) unsigned char bkc_smem[];
  __shared__ int64_t s_win;
  const int t = threadIdx.x, g = t & 31;
  for (;;) {
    if (t == 0) s_win = (int64_t)atomicAdd(ctr, 1ull) * 32;
    __syncthreads();
    const int64_t win = s_win;
    __syncthreads();
    if (win >= N) break;
    const int64_t mine = win + g;
    int64_t my_lo = 0, my_len = 0;
    if (mine < N) { my_lo = off[mine]; my_len = off[mine + 1] - my_lo; }
    uint32_t mask = __ballot_sync(0xffffffffu, mine < N && my_len > LO && my_len <= HI);  // same in every warp
    while (mask) {
      const int pos = __ffs(mask) - 1;
      mask &= mask - 1;
      const int64_t lo = __shfl_sync(0xffffffffu, my_lo, pos);
      const int len = (int)__shfl_sync(0xffffffffu, my_len, pos);
      bucket_sort_cta<W, false>(d + lo, len, bkc_smem, one);
    }
  }
}

}  // namespace gas
