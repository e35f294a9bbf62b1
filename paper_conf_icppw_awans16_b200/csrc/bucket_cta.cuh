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

// One array per CTA of WR warps (T = 32 WR threads, 32 keys per thread,
// n <= 1024 WR); W = the power of two >= WR whose whole-array network is the
// fallback (sort_cta with W - WR virtual padding warps, warp1024.cuh).
template <int W, int WR = W>
struct BkCta {
  static_assert(WR <= W && 2 * WR > W, "W = the power of two covering WR");
  static constexpr int T = 32 * WR;        // threads
  static constexpr int P = 1024 * WR;      // capacity (keys)
  static constexpr int ROWS = 64 * WR;     // bucket rows = buckets 0 .. ROWS-1
  static constexpr int CNT_BYTES = ROWS * 4;
  static constexpr int SLOT_BYTES = ROWS * kBkRowWords * 4;
  // the fallback network needs 1024 W words of exchange + 4 KB per warp
  static constexpr int FB_BYTES = 1024 * W * 4 + WR * 4096;
  static constexpr int BUF_BYTES = SLOT_BYTES > FB_BYTES ? SLOT_BYTES : FB_BYTES;
  // cross-warp scratch: raw-bit min/max [0, 2 WR), key min/max [32, 32 + 2 WR), scan partials [64, 64 + WR)
  static constexpr int RED_BYTES = 96 * 4;
  static constexpr int SMEM = CNT_BYTES + BUF_BYTES + RED_BYTES;
  static_assert(WR <= 16, "cross-warp scratch");
};

// Resident warps per SM (the register budget follows), measured: WR = 2: 18
// (n = 2000: 4.69 ms vs 4.85 at 16, 4.77 at 20); WR = 3: 21 (n = 2500: 5.50 vs
// 5.69 at 18); WR = 1, 4: 20 (SMEM caps WR = 4 at 20).
#ifdef GAS_BKC_WARPS_PER_SM
template <int WR> __host__ __device__ constexpr int bkc_warps_per_sm() { return GAS_BKC_WARPS_PER_SM; }
#else
#ifndef GAS_BKC_W2
#define GAS_BKC_W2 18
#endif
#ifndef GAS_BKC_W3
#define GAS_BKC_W3 21
#endif
template <int WR> __host__ __device__ constexpr int bkc_warps_per_sm() { return WR == 2 ? GAS_BKC_W2 : (WR == 3 ? GAS_BKC_W3 : (WR >= 8 ? 16 : 20)); }
#endif
template <int WR> __host__ __device__ constexpr int bkc_min_blocks() { return bkc_warps_per_sm<WR>() / WR > 0 ? bkc_warps_per_sm<WR>() / WR : 1; }

// Sort the n keys at `arr` (P/2 < n <= P; VEC: 16-byte-aligned, n % 4 == 0)
// in place. All T threads of the CTA call it; `sm` is BkCta<W, WR>::SMEM bytes.
// The steps are those of k_fixed_bucket1024 (bucket1024.cuh): counters start
// at their rows' addresses so the atomic returns the slot address, fused
// scatter, pads only after each row's last key, gathers of the occupied
// chunks (upper buckets first, their sorted keys then pad the lower round),
// output staged over the drained rows T .. 2T-1.
#ifndef GAS_BKC_PREFETCH
#define GAS_BKC_PREFETCH 1
#endif
#ifndef GAS_BKC_TMA_STORE  // output of the CTA bucket path through one TMA bulk store (see bucket_sort_cta)
#define GAS_BKC_TMA_STORE 1
#endif

// Arrays per CTA: GROUPS independent thread groups of WR warps share one CTA
// (one CTA per SM; GAS_BKC_GROUPS=0: one group per CTA, several CTAs per SM)
// and synchronise with their own named barrier (group_sync, bitonic.cuh).
#ifndef GAS_BKC_GROUPS
#define GAS_BKC_GROUPS 1
#endif
// Measured (1 B200): grouped n=2500 5.76 -> 5.69 ms, 4000 5.07 -> 5.00, 8000
// 6.39 -> 6.32, but n=2000 (WR = 2) 4.86 -> 5.14: groups for WR >= 3 only.
template <int WR> __host__ __device__ constexpr bool bkc_grouped() { return GAS_BKC_GROUPS && WR >= 3; }
template <int WR> __host__ __device__ constexpr int bkc_groups() { return bkc_grouped<WR>() ? bkc_min_blocks<WR>() : 1; }
template <int WR> __host__ __device__ constexpr int bkc_block() { return 32 * WR * bkc_groups<WR>(); }
template <int WR> __host__ __device__ constexpr int bkc_launch_min_blocks() { return bkc_grouped<WR>() ? 1 : bkc_min_blocks<WR>(); }
static_assert(bkc_groups<2>() <= 15 && bkc_groups<3>() <= 15, "named barriers 1..15");

// Barrier of the group (WR == 1: the warp).
template <int WR>
__device__ __forceinline__ void bar_cta(uint32_t bar) {
  if constexpr (WR > 1) group_sync(bar);
  else __syncwarp();
}

// t = thread index in the group (0 .. 32 WR - 1); bar = the group's barrier
// (0: the group is the whole CTA).
// RV: key slots r < RV are always inside the array (n > 32 WR RV; 16 for the
// classes (P/2, P], 8 when the W = 1 kernel serves 256 < n <= 512).
// TMA: the bucket path's output leaves through one TMA bulk store of the
// staged array (thread 0 of the group issues it; the sorted key i is staged at
// word i + head, head = the array's word offset inside its 16-byte chunk, so
// that shared source and global destination share their alignment; the <= 3
// words before the first and after the last 16-byte boundary are stored one by
// one). Thread 0 waits for the previous store's reads before the group's first
// row write of the next array; the kernel waits for completion before exiting.
#ifndef GAS_BKC_VOTE_MERGE
#define GAS_BKC_VOTE_MERGE 1
#endif
constexpr uint32_t kBkcOverflow = 0xFFFFFFFFu;  // a warp's scan total when one of its buckets overflowed (totals < 2^31)
// MASK: staging stores under bitmask predicates (stage_first, bucket1024.cuh):
// measured faster for one array per CTA (n = 2000 4.60 -> 4.54 ms, configs[3]
// 5.70 -> 5.68) and slower for the grouped CTAs (n = 4000 4.82 -> 5.08).
template <int W, int WR, bool VEC, int RV = 16, bool TMA = (GAS_BKC_TMA_STORE != 0), bool MASK = (GAS_BK_MASKSTORE != 0)>
__device__ __forceinline__ void bucket_sort_cta(uint32_t* __restrict__ arr, int n, unsigned char* sm, uint32_t one,
                                                int t, uint32_t bar) {
  using C = BkCta<W, WR>;
  constexpr int T = C::T;
  const int lane = t & 31, warp = t >> 5;
  const uint32_t cnt_sa = (uint32_t)__cvta_generic_to_shared(sm);
  const uint32_t slot_sa = cnt_sa + C::CNT_BYTES;
  const uint32_t stage_sa = slot_sa + T * kBkRowWords * 4;  // output word p at stage_sa + 4p (rows T .. 2T-1)
  const uint32_t slot_last = slot_sa + C::SLOT_BYTES - 4;
  unsigned char* const slot_ptr = sm + C::CNT_BYTES;
  uint32_t* const red = reinterpret_cast<uint32_t*>(sm + C::CNT_BYTES + C::BUF_BYTES);
  const uint32_t cnt_b0 = cnt_sa - 0x4B000000u * 4u;
  const uint32_t row0 = slot_sa + t * (kBkRowWords * 4);  // rows of buckets t and t + T
  const uint32_t row1 = row0 + T * (kBkRowWords * 4);
  const int nc = n >> 2;
  const int head = TMA ? (int)((reinterpret_cast<uintptr_t>(arr) >> 2) & 3u) : 0;  // staging shift (0 when VEC)
  if (TMA && warp == 0) bulk_wait_read_elect();  // thread 0 (the issuing lane); ordered by the first barrier
  // key r of this thread: VEC element 4 (t + T (r/4)) + r%4, else element t + T r
  auto valid = [&](int r) -> bool {
    if (VEC) return (r >> 2) < 4 || t + T * (r >> 2) < nc;
    return r < RV || t + T * r < n;
  };

  // ---- stage in (raw bits); slots past the end repeat k[0] (always valid)
  uint32_t k[32];
  if constexpr (VEC) {
    const uint4* src = reinterpret_cast<const uint4*>(arr);
#pragma unroll
    for (int q = 0; q < 8; ++q) {
      const uint4 v = q < 4 ? ld_stream(src + t + T * q) : ldg_cs_if(valid(4 * q), src + t + T * q);
      k[4 * q] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
    }
  } else {
#pragma unroll
    for (int r = 0; r < 32; ++r) k[r] = valid(r) ? ld_stream(arr + t + T * r) : 0u;
  }
#pragma unroll
  for (int r = VEC ? 16 : RV; r < 32; ++r) k[r] = valid(r) ? k[r] : k[0];
  // ---- min / max of the raw bits, then (if needed) of the keys, across the CTA
  uint32_t umin = k[0], umax = k[0];
#pragma unroll
  for (int r = 1; r < 31; r += 2) {
    umin = __vimin3_u32(umin, k[r], k[r + 1]);
    umax = __vimax3_u32(umax, k[r], k[r + 1]);
  }
  umin = __reduce_min_sync(0xffffffffu, min(umin, k[31]));
  umax = __reduce_max_sync(0xffffffffu, max(umax, k[31]));
  // Barriers: 5 or 6 per array. The previous array's last shared accesses (output
  // staging reads) are ordered before this array's first row write by the
  // barrier below; counters and `red` were last read several barriers ago.
  sts32(cnt_sa + t * 4, row0);  // counter b starts at the address of row b
  sts32(cnt_sa + (T + t) * 4, row1);
  if constexpr (WR > 1) {
    if (lane == 0) { red[2 * warp] = umin; red[2 * warp + 1] = umax; }
  }
  bar_cta<WR>(bar);
  if constexpr (WR > 1) {
#pragma unroll
    for (int w = 0; w < WR; ++w) { umin = min(umin, red[2 * w]); umax = max(umax, red[2 * w + 1]); }
  }
  const bool raw = umin > 0u && umax < 0x7F800000u;  // every value positive and finite (CTA-uniform)
  bool use_buckets = true;
  if (!raw) {
    uint32_t kmin = 0xFFFFFFFFu, kmax = 0u;
#pragma unroll
    for (int r = 0; r < 32; ++r) {
      const uint32_t kk = key_from_bits(k[r]);
      kmin = min(kmin, kk);
      kmax = max(kmax, kk);
    }
    kmin = __reduce_min_sync(0xffffffffu, kmin);
    kmax = __reduce_max_sync(0xffffffffu, kmax);
    if constexpr (WR > 1) {
      if (lane == 0) { red[32 + 2 * warp] = kmin; red[32 + 2 * warp + 1] = kmax; }
      group_sync(bar);
#pragma unroll
      for (int w = 0; w < WR; ++w) { kmin = min(kmin, red[32 + 2 * w]); kmax = max(kmax, red[32 + 2 * w + 1]); }
    }
    use_buckets = kmin > 0x007FFFFFu && kmax < 0xFF800000u;  // no infinity, no NaN
    umin = bits_from_key(kmin);
    umax = bits_from_key(kmax);
  }
  const float vmin = __uint_as_float(umin), vmax = __uint_as_float(umax);
  const float range = __fsub_rn(vmax, vmin);
  const float s = __fdiv_rn((float)(C::ROWS - 1), range);
  use_buckets = use_buckets && range > 0.0f && range <= 3.402823466e38f && s <= 3.402823466e38f;
  uint32_t t0 = 0, t1 = 0, base0 = 0, base1 = 0;
  if (use_buckets) {  // CTA-uniform
    if (raw) {
#pragma unroll
      for (int g = 0; g < 32; g += 4) {
        uint32_t sa[4];
#pragma unroll
        for (int r = g; r < g + 4; ++r) sa[r - g] = atoms_add4_if(valid(r), bucket_bits(k[r], vmin, s) * 4u + cnt_b0);
#pragma unroll
        for (int r = g; r < g + 4; ++r) sts32_if(valid(r), min(sa[r - g], slot_last), k[r]);
      }
    } else {
#pragma unroll
      for (int g = 0; g < 32; g += 4) {
        uint32_t sa[4];
#pragma unroll
        for (int r = g; r < g + 4; ++r) sa[r - g] = atoms_add4_if(valid(r), bucket_bits(k[r], vmin, s) * 4u + cnt_b0);
#pragma unroll
        for (int r = g; r < g + 4; ++r) sts32_if(valid(r), min(sa[r - g], slot_last), key_from_bits(k[r]));
      }
    }
    bar_cta<WR>(bar);
    t0 = (lds32(cnt_sa + t * 4) - row0) >> 2;
    t1 = (lds32(cnt_sa + (T + t) * 4) - row1) >> 2;
    // overflow vote and bucket bases share one barrier: a warp whose buckets
    // fit posts its scan total, one that overflows posts kBkcOverflow
    // (GAS_BKC_VOTE_MERGE=0: a separate bar.red.and vote first)
    if constexpr (WR > 1 && !GAS_BKC_VOTE_MERGE) use_buckets = group_and(t0 <= 32u && t1 <= 32u, bar);
    else use_buckets = __all_sync(0xffffffffu, t0 <= 32u && t1 <= 32u);
    uint32_t x = 0, before = 0, total = 0;
    if (use_buckets) {
#pragma unroll
      for (int j = 0; j < 3; ++j) {
        sts32_if(((t0 + j) & 3u) != 0u, row0 + (t0 + j) * 4, kPadKey);
        sts32_if(((t1 + j) & 3u) != 0u, row1 + (t1 + j) * 4, kPadKey);
      }
      // bucket bases: exclusive scan of the 2T bucket sizes (two 16-bit halves)
      x = t0 | (t1 << 16);
#pragma unroll
      for (int m = 1; m < 32; m <<= 1) {
        const uint32_t y = __shfl_up_sync(0xffffffffu, x, m);
        if (lane >= m) x += y;
      }
      total = __shfl_sync(0xffffffffu, x, 31);
    }
    if constexpr (WR > 1 && GAS_BKC_VOTE_MERGE) {
      uint32_t* const part = red + 64;
      if (lane == 31) part[warp] = use_buckets ? x : kBkcOverflow;
      group_sync(bar);  // also publishes the pads
      total = 0;
#pragma unroll
      for (int w = 0; w < WR; ++w) {
        const uint32_t pw = part[w];
        use_buckets = use_buckets && pw != kBkcOverflow;
        before += (w < warp) ? pw : 0u;
        total += pw;
      }
    }
    if (use_buckets) {
      if constexpr (WR > 1 && !GAS_BKC_VOTE_MERGE) {
        uint32_t* const part = red + 64;
        if (lane == 31) part[warp] = x;
        group_sync(bar);  // also publishes the pads
        total = 0;
#pragma unroll
        for (int w = 0; w < WR; ++w) {
          const uint32_t pw = part[w];
          before += (w < warp) ? pw : 0u;
          total += pw;
        }
      }
      else __syncwarp();  // publishes the pads
      x += before;
      base0 = (x & 0xFFFFu) - t0;
      base1 = (total & 0xFFFFu) + (x >> 16) - t1;
    }
  }

  if (use_buckets) {
    // two rounds: bucket t + T, then bucket t
#pragma unroll 1
    for (int rho = 0; rho < 2; ++rho) {
      const uint32_t tb = rho ? t0 : t1;
      const uint32_t row = rho ? row0 : row1;
      const uint32_t ob = stage_sa + ((rho ? base0 : base1) + head) * 4;
      if (rho == 0) {
#pragma unroll
        for (int i = 0; i < 32; ++i) k[i] = kPadKey;
      }
#pragma unroll
      for (int q = 0; q < 8; ++q) lds128_if(4u * q < tb, row + q * 16, k[4 * q], k[4 * q + 1], k[4 * q + 2], k[4 * q + 3]);
      // rows T .. 2T-1 are drained before any output is staged over them (the
      // second round reads rows 0 .. T-1, which staging never touches)
      if (rho == 0) bar_cta<WR>(bar);
      sortn_bk<32>(k, one);
      if (MASK) {  // bitmask predicates (R2P; stage_first, bucket1024.cuh)
        uint32_t* const sw = reinterpret_cast<uint32_t*>(sm);
        if (TMA && !raw) stage_first<true>(sw, (ob - cnt_sa) >> 2, tb, k);
        else stage_first<false>(sw, (ob - cnt_sa) >> 2, tb, k);
      } else if (TMA && !raw) {  // the bulk store copies bits: stage transformed keys (k keeps the keys: the
#pragma unroll            // second round uses them as padding)
        for (int i = 0; i < 32; ++i) sts32_if((uint32_t)i < tb, ob + i * 4, bits_from_key(k[i]));
      } else {
#pragma unroll
        for (int i = 0; i < 32; ++i) sts32_if((uint32_t)i < tb, ob + i * 4, k[i]);
      }
    }
    if constexpr (TMA) {
      asm volatile("fence.proxy.async.shared::cta;" ::: "memory");  // this thread's staging writes -> async proxy
      bar_cta<WR>(bar);
      const int h0 = (4 - head) & 3, h1 = h0 + ((n - h0) & ~3);  // [h0, h1): 16-byte aligned in both memories
      if (warp == 0 && h1 > h0)  // one elected lane of warp 0 (thread 0, which also waits for it)
        bulk_store_elect(arr + h0, stage_sa + (uint32_t)(head + h0) * 4u, (uint32_t)(h1 - h0) * 4u);
      if (t < h0) st_stream(arr + t, lds32(stage_sa + (head + t) * 4));
      else if (t >= 4 && t - 4 + h1 < n) st_stream(arr + (t - 4 + h1), lds32(stage_sa + (head + t - 4 + h1) * 4));
    } else {
    bar_cta<WR>(bar);
    if constexpr (VEC) {
      uint4* dst = reinterpret_cast<uint4*>(arr);
#pragma unroll
      for (int q = 0; q < 8; ++q) {
        const int c = t + T * q;
        uint4 v = lds128(stage_sa + c * 16);
        if (!raw) { v.x = bits_from_key(v.x); v.y = bits_from_key(v.y); v.z = bits_from_key(v.z); v.w = bits_from_key(v.w); }
        stg_cs_if(q < 4 || c < nc, dst + c, v);
      }
    } else {
      if (raw) {
#pragma unroll
        for (int r = 0; r < 32; ++r) {
          const int e = t + T * r;
          if (e < n) st_stream(arr + e, lds32(stage_sa + e * 4));
        }
      } else {
#pragma unroll
        for (int r = 0; r < 32; ++r) {
          const int e = t + T * r;
          if (e < n) st_stream(arr + e, bits_from_key(lds32(stage_sa + e * 4)));
        }
      }
    }
    }  // !TMA
  } else {
    // ---- fallback: the whole-array network (warp1024.cuh sort_cta)
#pragma unroll
    for (int r = 0; r < 32; ++r) k[r] = valid(r) ? key_from_bits(k[r]) : kPadKey;
    uint32_t* xs = reinterpret_cast<uint32_t*>(slot_ptr);
    uint32_t* wbuf = xs + 1024 * W + warp * 1024;
    bar_cta<WR>(bar);
    fill_virtual<W, WR>(xs, t);
    sort_cta<W>(k, t, lane, xs, wbuf, one, bar);
    bar_cta<WR>(bar);
    uint4* sb = reinterpret_cast<uint4*>(slot_ptr);
    stage_out_words<32>(k, sb, t * 32);
    bar_cta<WR>(bar);
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
  // no trailing barrier: the next array's first shared write to the rows
  // follows its first barrier (see above)
}

// Fixed length, one array per CTA (persistent grid-stride).
template <int W, int WR, bool VEC>
__global__ void __launch_bounds__(bkc_block<WR>(), bkc_launch_min_blocks<WR>())
    k_fixed_bucket_cta(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one) {
  extern __shared__ __align__(16) unsigned char bkc_smem[];
  constexpr int GR = bkc_groups<WR>();
  const int grp = threadIdx.x / (32 * WR), t = threadIdx.x % (32 * WR);
  const uint32_t bar = GR > 1 ? (uint32_t)(grp + 1) | ((uint32_t)(32 * WR) << 8) : 0u;
  unsigned char* const sm = bkc_smem + grp * BkCta<W, WR>::SMEM;
  const int64_t stride = (int64_t)gridDim.x * GR;
  for (int64_t a = (int64_t)blockIdx.x * GR + grp; a < N; a += stride) {
#if GAS_BKC_PREFETCH
    if (t < 32) prefetch_l2_elect(a + stride < N, d + (a + stride) * (int64_t)n, n);
#endif
    bucket_sort_cta<W, WR, VEC, 16, (GAS_BKC_TMA_STORE != 0), (GAS_BK_MASKSTORE != 0) && !bkc_grouped<WR>()>(
        d + a * (int64_t)n, n, sm, one, t, bar);
  }
  if (GAS_BKC_TMA_STORE && t == 0) asm volatile("cp.async.bulk.wait_group 0;" ::: "memory");
}

// Variable length: the arrays with LO < len <= HI (P/2 <= LO, HI <= P), found
// by scanning windows of 32 arrays handed out dynamically through `ctr` (one
// counter per launch, zeroed by the host), as k_offsets_cta. Rows may start
// at any 4-byte boundary: scalar loads and stores.
// (One group per CTA here: several small CTAs per SM co-reside with the other
// size classes' launches on the forked streams; grouped CTAs measured slower on
// configs[3], 6.13 vs 6.05 ms.)
template <int W, int WR, int RV = 16>
__global__ void __launch_bounds__(32 * WR, bkc_min_blocks<WR>())
    k_offsets_bucket(uint32_t* __restrict__ d, const int64_t* __restrict__ off, int64_t N, int64_t LO, int64_t HI,
                     unsigned long long* __restrict__ ctr, uint32_t one) {
  extern __shared__ __align__(16) unsigned char bkc_smem[];
  constexpr int GR = 1;
  __shared__ int64_t s_win[GR];
  const int grp = threadIdx.x / (32 * WR), t = threadIdx.x % (32 * WR), g = t & 31;
  const uint32_t bar = GR > 1 ? (uint32_t)(grp + 1) | ((uint32_t)(32 * WR) << 8) : 0u;
  unsigned char* const sm = bkc_smem + grp * BkCta<W, WR>::SMEM;
  for (;;) {
    if (t == 0) s_win[grp] = (int64_t)atomicAdd(ctr, 1ull) * 32;
    bar_cta<WR>(bar);
    const int64_t win = s_win[grp];
    bar_cta<WR>(bar);
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
#if GAS_BKC_PREFETCH
      if (mask) {  // warm L2 with the window's next array of this class
        const int nx = __ffs(mask) - 1;
        const int64_t nlo = __shfl_sync(0xffffffffu, my_lo, nx);
        const int64_t nlen = __shfl_sync(0xffffffffu, my_len, nx);
        if (t < 32) prefetch_l2_elect(true, d + nlo, nlen);
      }
#endif
      bucket_sort_cta<W, WR, false, RV>(d + lo, len, sm, one, t, bar);
    }
  }
  if (GAS_BKC_TMA_STORE && t == 0) asm volatile("cp.async.bulk.wait_group 0;" ::: "memory");
}

}  // namespace gas
