// bucket512.cuh — the bucket-then-network sort of bucket1024.cuh for arrays of
// 256 < n <= 512 keys (16-byte-aligned rows), one warp per array: 32 value
// buckets, one bucket (<= 32 keys, ~8-16 on flat data) per lane, one round of
// the 191-comparator network — about half the compare-exchanges of the
// 512-key bitonic network that sorts this class otherwise (segsort.cuh,
// G = 16). Same steps and correctness argument as k_fixed_bucket1024: the
// atomic returns the slot address, pads after each row's keys, occupied-chunk
// gathers into pad-preset registers, output staged over the drained rows,
// warp-uniform fallback to the (padded) 1024-key network.
#pragma once
#include <cstdint>

#include "bucket1024.cuh"
#include "segsort.cuh"

namespace gas {

#ifndef GAS_BK5_WARPS
#define GAS_BK5_WARPS 24  // warps per SM = per block (one block per SM); measured (round 2 build): 24 vs 20 vs 16 warps: n = 500 4.197 / 4.213 / 4.260 ms, n = 300 6.072 / 6.124 / 6.198
#endif
#ifndef GAS_BK5_NET16
// k_fixed_bucket512<NET16 = true> for n <= kBk5Net16MaxN: when every bucket of
// the warp holds <= 16 keys, the 63-comparator network on k[0..15] instead of
// 191 (the branch alone costs ~5% where most warps need 32 keys)
#define GAS_BK5_NET16 1
#endif
constexpr int kBk5Net16MaxN = 336;
constexpr int kBk5Block = 32 * GAS_BK5_WARPS;
constexpr int kBk5CntBytes = 32 * 4;
constexpr int kBk5SlotBytes = 32 * kBkRowWords * 4;  // also the fallback network's 4 KB scratch
constexpr int kBk5WarpBytes = kBk5CntBytes + kBk5SlotBytes;
constexpr int kBk5SmemBytes = GAS_BK5_WARPS * kBk5WarpBytes;

template <bool NET16>
__global__ void __launch_bounds__(kBk5Block, 1)
    k_fixed_bucket512(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one) {
  extern __shared__ __align__(16) uint4 bk5_smem[];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const uint32_t cnt_sa = (uint32_t)__cvta_generic_to_shared(bk5_smem) + warp * kBk5WarpBytes;
  const uint32_t slot_sa = cnt_sa + kBk5CntBytes;
  const uint32_t slot_last = slot_sa + kBk5SlotBytes - 4;
  uint32_t* const slot_ptr = reinterpret_cast<uint32_t*>(reinterpret_cast<unsigned char*>(bk5_smem) +
                                                         warp * kBk5WarpBytes + kBk5CntBytes);
  const int nc = n >> 2;  // 64 < nc <= 128
  const int64_t nwarps = (int64_t)gridDim.x * GAS_BK5_WARPS;
  const uint32_t cnt_b0 = cnt_sa - 0x4B000000u * 4u;
  const uint32_t row = slot_sa + lane * (kBkRowWords * 4);

  for (int64_t a = (int64_t)blockIdx.x * GAS_BK5_WARPS + warp; a < N; a += nwarps) {
    uint4* const dst = reinterpret_cast<uint4*>(d + a * (int64_t)n);
    uint32_t k[32];
#pragma unroll
    for (int q = 0; q < 4; ++q) {
      const int c = lane + 32 * q;
      const uint4 v = q < 2 ? ld_stream(dst + c) : ldg_cs_if(c < nc, dst + c);
      k[4 * q] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
    }
#if GAS_BK_PREFETCH
    bulk_prefetch_elect(a + nwarps < N, d + (a + nwarps) * (int64_t)n, (uint32_t)n * 4u);
#endif
#pragma unroll
    for (int q = 2; q < 4; ++q) {
      const bool v = lane + 32 * q < nc;
#pragma unroll
      for (int j = 0; j < 4; ++j) k[4 * q + j] = v ? k[4 * q + j] : k[0];
    }
    uint32_t umin = k[0], umax = k[0];
#pragma unroll
    for (int r = 1; r < 15; r += 2) {
      umin = __vimin3_u32(umin, k[r], k[r + 1]);
      umax = __vimax3_u32(umax, k[r], k[r + 1]);
    }
    umin = __reduce_min_sync(0xffffffffu, min(umin, k[15]));
    umax = __reduce_max_sync(0xffffffffu, max(umax, k[15]));
    const bool raw = umin > 0u && umax < 0x7F800000u;
    bool use_buckets = true;
    if (!raw) {
      uint32_t kmin = 0xFFFFFFFFu, kmax = 0u;
#pragma unroll
      for (int r = 0; r < 16; ++r) {
        const uint32_t kk = key_from_bits(k[r]);
        kmin = min(kmin, kk);
        kmax = max(kmax, kk);
      }
      kmin = __reduce_min_sync(0xffffffffu, kmin);
      kmax = __reduce_max_sync(0xffffffffu, kmax);
      use_buckets = kmin > 0x007FFFFFu && kmax < 0xFF800000u;
      umin = bits_from_key(kmin);
      umax = bits_from_key(kmax);
    }
    const float vmin = __uint_as_float(umin), vmax = __uint_as_float(umax);
    const float range = __fsub_rn(vmax, vmin);
    const float s = __fdiv_rn(31.0f, range);  // buckets 0 .. 31
    use_buckets = use_buckets && range > 0.0f && range <= 3.402823466e38f && s <= 3.402823466e38f;
    uint32_t t = 0, base = 0;
    if (use_buckets) {
      sts32(cnt_sa + lane * 4, row);
      __syncwarp();
      if (raw) {
#pragma unroll
        for (int g = 0; g < 16; g += 4) {
          uint32_t sa[4];
#pragma unroll
          for (int r = g; r < g + 4; ++r)
            sa[r - g] = atoms_add4_if((r >> 2) < 2 || lane + 32 * (r >> 2) < nc, bucket_bits(k[r], vmin, s) * 4u + cnt_b0);
#pragma unroll
          for (int r = g; r < g + 4; ++r) sts32_if((r >> 2) < 2 || lane + 32 * (r >> 2) < nc, min(sa[r - g], slot_last), k[r]);
        }
      } else {
#pragma unroll
        for (int g = 0; g < 16; g += 4) {
          uint32_t sa[4];
#pragma unroll
          for (int r = g; r < g + 4; ++r)
            sa[r - g] = atoms_add4_if((r >> 2) < 2 || lane + 32 * (r >> 2) < nc, bucket_bits(k[r], vmin, s) * 4u + cnt_b0);
#pragma unroll
          for (int r = g; r < g + 4; ++r)
            sts32_if((r >> 2) < 2 || lane + 32 * (r >> 2) < nc, min(sa[r - g], slot_last), key_from_bits(k[r]));
        }
      }
      __syncwarp();
      t = (lds32(cnt_sa + lane * 4) - row) >> 2;
      use_buckets = __all_sync(0xffffffffu, t <= 32u);
      if (use_buckets) {
#pragma unroll
        for (int j = 0; j < 3; ++j) sts32_if(((t + j) & 3u) != 0u, row + (t + j) * 4, kPadKey);
        uint32_t x = t;
#pragma unroll
        for (int m = 1; m < 32; m <<= 1) {
          const uint32_t y = __shfl_up_sync(0xffffffffu, x, m);
          if (lane >= m) x += y;
        }
        base = x - t;
        __syncwarp();
      }
    }
    if (use_buckets) {
#pragma unroll
      for (int i = 0; i < 32; ++i) k[i] = kPadKey;
#pragma unroll
      for (int q = 0; q < 8; ++q) lds128_if(4u * q < t, row + q * 16, k[4 * q], k[4 * q + 1], k[4 * q + 2], k[4 * q + 3]);
      __syncwarp();  // every row is drained before the output is staged over them
      if (NET16 && __all_sync(0xffffffffu, t <= 16u)) sortn_bk<16>(k, one);  // rows past 16 keep their pads
      else sortn_bk<32>(k, one);
      const uint32_t ob = slot_sa + base * 4;
      if (GAS_BK_MASKSTORE) {
        stage_first<false>(reinterpret_cast<uint32_t*>(bk5_smem), (ob - (uint32_t)__cvta_generic_to_shared(bk5_smem)) >> 2, t, k);
      } else {
#pragma unroll
        for (int i = 0; i < 32; ++i) sts32_if((uint32_t)i < t, ob + i * 4, k[i]);
      }
      __syncwarp();
      if (raw) {
#pragma unroll
        for (int q = 0; q < 4; ++q) {
          const int c = lane + 32 * q;
          stg_cs_if(q < 2 || c < nc, dst + c, lds128(slot_sa + c * 16));
        }
      } else {
#pragma unroll
        for (int q = 0; q < 4; ++q) {
          const int c = lane + 32 * q;
          uint4 v = lds128(slot_sa + c * 16);
          v.x = bits_from_key(v.x); v.y = bits_from_key(v.y); v.z = bits_from_key(v.z); v.w = bits_from_key(v.w);
          stg_cs_if(q < 2 || c < nc, dst + c, v);
        }
      }
    } else {
      // fallback: the data-oblivious 512-key bitonic network over the whole
      // warp (16 keys per lane, lane stages by shuffles; bitonic.cuh)
      __syncwarp();
      uint32_t k16[16];
#pragma unroll
      for (int r = 0; r < 16; ++r) {
        const bool v = (r >> 2) < 2 || lane + 32 * (r >> 2) < nc;
        k16[r] = v ? key_from_bits(k[r]) : kPadKey;
      }
      Bitonic<16, 32, 1>::sort(k16, lane, 0, nullptr, one);
      uint4* sb = reinterpret_cast<uint4*>(slot_ptr);
      stage_out_words<16>(k16, sb, lane * 16);
      __syncwarp();
#pragma unroll
      for (int q = 0; q < 4; ++q) {
        const int c = lane + 32 * q;
        if (c < nc) st_stream(dst + c, sb[swz(c)]);
      }
    }
    __syncwarp();
  }
}

// ---------------------------------------------------------------------------
// 128 < n <= 256 (16-byte-aligned rows): the same steps on a half warp per
// array (two arrays per warp): 16 value buckets per array, one bucket (<= 32
// keys, ~8-16 on flat data) per lane, one round of the 191-comparator network,
// against ~18 compare-exchanges per key of the 256-key bitonic network
// (segsort.cuh, G = 8) that sorts this class otherwise. Decisions that need
// warp-wide agreement (the fallback) are taken for both halves at once: if
// either array overflows a bucket, both take the 256-key bitonic network of
// their half (bitonic.cuh, G = 16).
#ifndef GAS_BK2_WARPS
#define GAS_BK2_WARPS 24
#endif
constexpr int kBk2Block = 32 * GAS_BK2_WARPS;
constexpr int kBk2HalfBytes = 16 * 4 + 16 * kBkRowWords * 4;  // counters + rows of one array
constexpr int kBk2SmemBytes = GAS_BK2_WARPS * 2 * kBk2HalfBytes;

static __global__ void __launch_bounds__(kBk2Block, 1)
    k_fixed_bucket256(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one) {
  extern __shared__ __align__(16) uint4 bk2_smem[];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const int hl = lane & 15, half = lane >> 4;
  const unsigned hmask = 0xFFFFu << (16 * half);
  const uint32_t cnt_sa = (uint32_t)__cvta_generic_to_shared(bk2_smem) + (warp * 2 + half) * kBk2HalfBytes;
  const uint32_t slot_sa = cnt_sa + 64;
  const uint32_t slot_last = slot_sa + 16 * kBkRowWords * 4 - 4;
  uint4* const sb = reinterpret_cast<uint4*>(reinterpret_cast<unsigned char*>(bk2_smem) + (warp * 2 + half) * kBk2HalfBytes + 64);
  const int nc = n >> 2;  // 32 < nc <= 64
  const int64_t nwarps = (int64_t)gridDim.x * GAS_BK2_WARPS;
  const uint32_t cnt_b0 = cnt_sa - 0x4B000000u * 4u;
  const uint32_t row = slot_sa + hl * (kBkRowWords * 4);

  for (int64_t w = (int64_t)blockIdx.x * GAS_BK2_WARPS + warp; 2 * w < N; w += nwarps) {
    const int64_t a = 2 * w + half;
    const bool live = a < N;
    uint4* const dst = reinterpret_cast<uint4*>(d + (live ? a : 0) * (int64_t)n);
    uint32_t k[32];
#pragma unroll
    for (int q = 0; q < 4; ++q) {
      const int c = hl + 16 * q;
      const uint4 v = ldg_cs_if(live && (q < 2 || c < nc), dst + c);
      k[4 * q] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
    }
#if GAS_BK_PREFETCH
    {  // the warp's next pair of arrays, one bulk prefetch by one elected lane
      const int64_t nb = 2 * (w + nwarps), cnt = N - nb < 2 ? N - nb : 2;
      bulk_prefetch_elect(nb < N, d + nb * (int64_t)n, (uint32_t)(cnt > 0 ? cnt : 0) * (uint32_t)n * 4u);
    }
#endif
#pragma unroll
    for (int q = 2; q < 4; ++q) {
      const bool v = hl + 16 * q < nc;
#pragma unroll
      for (int j = 0; j < 4; ++j) k[4 * q + j] = v ? k[4 * q + j] : k[0];
    }
    uint32_t umin = k[0], umax = k[0];
#pragma unroll
    for (int r = 1; r < 15; r += 2) {
      umin = __vimin3_u32(umin, k[r], k[r + 1]);
      umax = __vimax3_u32(umax, k[r], k[r + 1]);
    }
    umin = __reduce_min_sync(hmask, min(umin, k[15]));
    umax = __reduce_max_sync(hmask, max(umax, k[15]));
    const bool raw = umin > 0u && umax < 0x7F800000u;
    bool use_buckets = true;
    if (!raw) {
      uint32_t kmin = 0xFFFFFFFFu, kmax = 0u;
#pragma unroll
      for (int r = 0; r < 16; ++r) {
        const uint32_t kk = key_from_bits(k[r]);
        kmin = min(kmin, kk);
        kmax = max(kmax, kk);
      }
      kmin = __reduce_min_sync(hmask, kmin);
      kmax = __reduce_max_sync(hmask, kmax);
      use_buckets = kmin > 0x007FFFFFu && kmax < 0xFF800000u;
      umin = bits_from_key(kmin);
      umax = bits_from_key(kmax);
    }
    const float vmin = __uint_as_float(umin), vmax = __uint_as_float(umax);
    const float range = __fsub_rn(vmax, vmin);
    const float s = __fdiv_rn(15.0f, range);  // buckets 0 .. 15
    use_buckets = __all_sync(0xffffffffu, !live || (use_buckets && range > 0.0f && range <= 3.402823466e38f &&
                                                    s <= 3.402823466e38f));
    uint32_t t = 0, base = 0;
    if (use_buckets) {
      sts32(cnt_sa + hl * 4, row);
      __syncwarp();
#pragma unroll
      for (int g = 0; g < 16; g += 4) {
        uint32_t sa[4];
#pragma unroll
        for (int r = g; r < g + 4; ++r)
          sa[r - g] = atoms_add4_pred(live && ((r >> 2) < 2 || hl + 16 * (r >> 2) < nc), bucket_bits(k[r], vmin, s) * 4u + cnt_b0);
#pragma unroll
        for (int r = g; r < g + 4; ++r)
          sts32_if(live && ((r >> 2) < 2 || hl + 16 * (r >> 2) < nc), min(sa[r - g], slot_last), raw ? k[r] : key_from_bits(k[r]));
      }
      __syncwarp();
      t = (lds32(cnt_sa + hl * 4) - row) >> 2;
      use_buckets = __all_sync(0xffffffffu, t <= 32u);
      if (use_buckets) {
#pragma unroll
        for (int j = 0; j < 3; ++j) sts32_if(((t + j) & 3u) != 0u, row + (t + j) * 4, kPadKey);
        uint32_t x = t;
#pragma unroll
        for (int m = 1; m < 16; m <<= 1) {
          const uint32_t y = __shfl_up_sync(0xffffffffu, x, m, 16);
          if (hl >= m) x += y;
        }
        base = x - t;
        __syncwarp();
      }
    }
    if (use_buckets) {
#pragma unroll
      for (int i = 0; i < 32; ++i) k[i] = kPadKey;
#pragma unroll
      for (int q = 0; q < 8; ++q) lds128_if(4u * q < t, row + q * 16, k[4 * q], k[4 * q + 1], k[4 * q + 2], k[4 * q + 3]);
      __syncwarp();  // every row is drained before the output is staged over them
      sortn_bk<32>(k, one);
      const uint32_t ob = slot_sa + base * 4;
      if (GAS_BK_MASKSTORE) {
        stage_first<false>(reinterpret_cast<uint32_t*>(bk2_smem), (ob - (uint32_t)__cvta_generic_to_shared(bk2_smem)) >> 2, t, k);
      } else {
#pragma unroll
        for (int i = 0; i < 32; ++i) sts32_if((uint32_t)i < t, ob + i * 4, k[i]);
      }
      __syncwarp();
#pragma unroll
      for (int q = 0; q < 4; ++q) {
        const int c = hl + 16 * q;
        uint4 v = lds128(slot_sa + c * 16);
        if (!raw) { v.x = bits_from_key(v.x); v.y = bits_from_key(v.y); v.z = bits_from_key(v.z); v.w = bits_from_key(v.w); }
        stg_cs_if(live && (q < 2 || c < nc), dst + c, v);
      }
    } else {
      // fallback (either array of the warp): the 256-key bitonic network of each half
      __syncwarp();
      uint32_t k16[16];
#pragma unroll
      for (int r = 0; r < 16; ++r) {
        const bool v = (r >> 2) < 2 || hl + 16 * (r >> 2) < nc;
        k16[r] = v ? key_from_bits(k[r]) : kPadKey;
      }
      Bitonic<16, 16, 1>::sort(k16, hl, 0, nullptr, one);
      stage_out_words<16>(k16, sb, hl * 16);
      __syncwarp();
#pragma unroll
      for (int q = 0; q < 4; ++q) {
        const int c = hl + 16 * q;
        if (live && c < nc) st_stream(dst + c, sb[swz(c)]);
      }
    }
    __syncwarp();
  }
}

}  // namespace gas
