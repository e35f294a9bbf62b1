// segsort.cuh — the segment-sort kernels.
//
// One kernel instantiation per size class P = 2^p >= n (row a4). Each array
// is owned by a group of G lanes (P <= 1024: several arrays per warp) or by a
// CTA of W warps (P = 2048, 4096) — the paper's "each block is assigned one
// array" at the granularity that fits the array. Per array:
//   a2 stage in   HBM -> registers, coalesced (LDG.128 when 16-B aligned)
//   a3 transform  float bits -> ordered uint32 key (ordered_key.cuh)
//   a4 pad        slots n..P-1 = kPadKey
//   a5 sort       bitonic network (bitonic.cuh)
//   a6 inverse    key -> float bits
//   a7 store      registers -> swizzled shared memory -> coalesced in-place
//                 store (STG.128 when aligned); every byte is written once,
//                 only inside the array's own range.
// Kernels are persistent (grid-stride over arrays) so that the grid is a
// multiple of the 148 SMs' resident blocks. Zero device workspace.
#pragma once
#include <cstdint>

#include "bitonic.cuh"
#include "ordered_key.cuh"
#include "warp1024.cuh"
#include "bulk.cuh"

namespace gas {

#ifndef GAS_WARP_BLOCK
#define GAS_WARP_BLOCK 256
#endif
constexpr int kWarpBlock = GAS_WARP_BLOCK;  // threads per block for the warp-level classes
#ifndef GAS_WARP_WARPS_PER_SM
#define GAS_WARP_WARPS_PER_SM 16  // occupancy target of the warp classes: 16 warps/SM -> up to 128 registers
#endif
#ifndef GAS_WARP_MIN_BLOCKS
#define GAS_WARP_MIN_BLOCKS (GAS_WARP_WARPS_PER_SM * 32 / GAS_WARP_BLOCK)
#endif

#ifndef GAS_SMALL_PREFETCH
#define GAS_SMALL_PREFETCH 1
#endif

// Occupancy target per class (blocks of kWarpBlock threads per SM), measured
// on B200 (profiles/r01_variants_small_occupancy.txt): the 1024 class (G = 32)
// and the 256 class (G = 8) run best at 2 blocks (<= 128 registers), the
// others at 3 blocks (<= 85 registers, small spills).
__host__ __device__ constexpr int warp_min_blocks(int G) { return (G == 32 || G == 8) ? GAS_WARP_MIN_BLOCKS : GAS_WARP_MIN_BLOCKS + 1; }
// GAS_WARP_BIG: the same warps per SM as one block (warp_min_blocks(G) x
// kWarpBlock threads) instead of several kWarpBlock-thread blocks (the bucket
// kernel measured 4.22 vs 4.39 ms for one 768-thread block per SM).
#ifndef GAS_WARP_BIG
#define GAS_WARP_BIG 1
#endif
// Measured (configs[1] shape, 1 B200): n=500 6.52 -> 6.16 ms, n=250 6.11 -> 5.89,
// n=100 4.77 -> 4.53, but n=60 (G = 2) 3.34 -> 3.59: classes with G >= 4 only.
template <int G> __host__ __device__ constexpr bool warp_big() { return GAS_WARP_BIG && G >= 4; }
template <int G> __host__ __device__ constexpr int warp_block() { return warp_big<G>() ? warp_min_blocks(G) * kWarpBlock : kWarpBlock; }
template <int G> __host__ __device__ constexpr int warp_block_min() { return warp_big<G>() ? 1 : warp_min_blocks(G); }
template <int KPT> __host__ __device__ constexpr int warp_smem_chunks() { return 32 * KPT / 4 > 0 ? 32 * KPT / 4 : 1; }  // uint4 per warp
template <int KPT, int G> __host__ __device__ constexpr int warp_smem_bytes() { return warp_block<G>() / 32 * warp_smem_chunks<KPT>() * 16; }

// XOR swizzle of 16-byte chunks inside 128-byte rows: chunk c of a rank-order
// buffer lives at physical chunk swz(c). Writes of 8 consecutive chunks per
// thread and reads of 32 consecutive chunks per warp are both conflict-free.
__device__ __forceinline__ int swz(int c) { return (c & ~7) | ((c ^ (c >> 3)) & 7); }

__device__ __forceinline__ uint4 ld_stream(const uint4* p) { return __ldcs(p); }
__device__ __forceinline__ uint32_t ld_stream(const uint32_t* p) { return __ldcs(p); }
__device__ __forceinline__ void st_stream(uint4* p, uint4 v) { __stcs(p, v); }
__device__ __forceinline__ void st_stream(uint32_t* p, uint32_t v) { __stcs(p, v); }

// ---- a2-a4: load one array's n elements into KPT keys per thread ----------
// Element (or 16-byte chunk) e of the array goes to thread (e % TH), slot
// e / TH; which slot holds which input element is irrelevant to a sort.
template <int KPT, int TH, bool VEC>
__device__ __forceinline__ void load_keys(uint32_t (&k)[KPT], const uint32_t* __restrict__ src, int n, int tid,
                                          bool valid) {
  if constexpr (VEC) {
    const uint4* s4 = reinterpret_cast<const uint4*>(src);
    const int nc = n >> 2;
#pragma unroll
    for (int q = 0; q < KPT / 4; ++q) {
      const int c = tid + TH * q;
      uint4 v = make_uint4(kPadKey, kPadKey, kPadKey, kPadKey);
      if (valid && c < nc) {
        v = ld_stream(s4 + c);
        v.x = key_from_bits(v.x); v.y = key_from_bits(v.y);
        v.z = key_from_bits(v.z); v.w = key_from_bits(v.w);
      }
      k[4 * q + 0] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
    }
  } else {
#pragma unroll
    for (int q = 0; q < KPT; ++q) {
      const int e = tid + TH * q;
      k[q] = (valid && e < n) ? key_from_bits(ld_stream(src + e)) : kPadKey;
    }
  }
}

// ---- a6-a7 (part 1): thread holding ranks [tid*KPT, tid*KPT+KPT) writes
// them, decoded, into the rank-order swizzled buffer `sb` (16-byte chunks).
template <int KPT>
__device__ __forceinline__ void stage_out(const uint32_t (&k)[KPT], uint4* sb, int chunk0) {
  static_assert(KPT >= 4, "vector staging needs 4 keys per thread");
#pragma unroll
  for (int q = 0; q < KPT / 4; ++q)
    sb[swz(chunk0 + q)] = make_uint4(bits_from_key(k[4 * q]), bits_from_key(k[4 * q + 1]),
                                     bits_from_key(k[4 * q + 2]), bits_from_key(k[4 * q + 3]));
}

__device__ __forceinline__ uint32_t sword(const uint4* sb, int w) {
  return reinterpret_cast<const uint32_t*>(sb)[swz(w >> 2) * 4 + (w & 3)];
}
__device__ __forceinline__ void sword_set(uint4* sb, int w, uint32_t v) {
  reinterpret_cast<uint32_t*>(sb)[swz(w >> 2) * 4 + (w & 3)] = v;
}

// Write KPT rank-consecutive keys starting at rank-word w0 (any KPT).
template <int KPT>
__device__ __forceinline__ void stage_out_words(const uint32_t (&k)[KPT], uint4* sb, int w0) {
  if constexpr (KPT >= 4) {
    stage_out<KPT>(k, sb, w0 >> 2);
  } else {
#pragma unroll
    for (int r = 0; r < KPT; ++r) sword_set(sb, w0 + r, bits_from_key(k[r]));
  }
}

// ===================================================== fixed-length kernels

// Warp-level classes: P = KPT * G <= 1024, GROUPS = 32 / G arrays per warp.
template <int KPT, int G, bool VEC>
__global__ void __launch_bounds__(warp_block<G>(), warp_block_min<G>()) k_fixed_warp(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one) {
  constexpr int GROUPS = 32 / G;
  constexpr int P = KPT * G;
  constexpr int BLK = warp_block<G>();
  extern __shared__ uint4 warp_dsm[];  // warp_smem_bytes<KPT, G>()
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const int g = lane & (G - 1), grp = lane / G;
  uint4* sb = warp_dsm + warp * warp_smem_chunks<KPT>();
  const int64_t nwarps = (int64_t)gridDim.x * (BLK / 32);
  for (int64_t base = ((int64_t)blockIdx.x * (BLK / 32) + warp) * GROUPS; base < N; base += nwarps * GROUPS) {
    const int64_t a = base + grp;
    const bool valid = a < N;
    uint32_t k[KPT];
    load_keys<KPT, G, VEC>(k, d + (valid ? a : 0) * (int64_t)n, n, g, valid);
#if GAS_SMALL_PREFETCH
    if constexpr (G >= 8 && G < 32) {
      // P = 256, 512: several arrays per warp, little work per byte, exposed to
      // HBM latency: warm L2 with the warp's next GROUPS arrays (one contiguous
      // TMA bulk prefetch issued by one lane). Measured: n=500 6.85 -> 6.35 ms;
      // no gain for the other classes (profiles/r01_variants_small_prefetch.txt).
      // (unaligned rows: only the 16-byte-aligned interior of the range)
      const int64_t nb = base + nwarps * GROUPS;
      const int64_t cnt = (N - nb < GROUPS) ? N - nb : GROUPS;
      const uintptr_t lo = (reinterpret_cast<uintptr_t>(d + nb * (int64_t)n) + 15) & ~uintptr_t(15);
      const uintptr_t hi = reinterpret_cast<uintptr_t>(d + (nb + cnt) * (int64_t)n) & ~uintptr_t(15);
      bulk_prefetch_elect(nb < N && hi > lo, reinterpret_cast<const void*>(lo), (uint32_t)(hi - lo));  // one elected lane
    }
#endif
    if constexpr (KPT == 32 && G >= 2) sort_group_warp<G>(k, g, reinterpret_cast<uint32_t*>(sb), one);
    else Bitonic<KPT, G, 1>::sort(k, g, 0, nullptr, one);
    stage_out_words<KPT>(k, sb, grp * P + g * KPT);
    __syncwarp();
    if constexpr (VEC) {
      // chunk c of the warp buffer = group c / (P/4), position (c % (P/4))*4
      const int nc = n >> 2;
#pragma unroll
      for (int q = 0; q < KPT / 4; ++q) {
        const int c = lane + 32 * q;
        const int gg = c / (P / 4), pc = c % (P / 4);
        const int64_t aa = base + gg;
        if (aa < N && pc < nc) st_stream(reinterpret_cast<uint4*>(d + aa * (int64_t)n) + pc, sb[swz(c)]);
      }
    } else {
#pragma unroll
      for (int q = 0; q < KPT; ++q) {
        const int w = lane + 32 * q;
        const int gg = w / P, pw = w % P;
        const int64_t aa = base + gg;
        if (aa < N && pw < n) st_stream(d + aa * (int64_t)n + pw, sword(sb, w));
      }
    }
    __syncwarp();
  }
}

// P = 1024 class with 16-byte-aligned rows (n % 4 == 0, aligned base): one
// warp per array; while the warp sorts array t its next array t+1 is already
// in flight into the warp's second shared-memory buffer by a TMA bulk copy
// (cp.async.bulk + mbarrier), so global-load latency is off the critical
// path. Dynamic shared memory: kWarpBlock/32 warps x 2 x 4 KB + barriers.
constexpr int kTmaSmemBytes = (kWarpBlock / 32) * 2 * 4096 + (kWarpBlock / 32) * 2 * 8;

static __global__ void __launch_bounds__(kWarpBlock, GAS_WARP_MIN_BLOCKS)
    k_fixed_1024_tma(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one) {
  extern __shared__ __align__(128) uint4 dsm[];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  uint4* buf0 = dsm + warp * 512;  // 2 x 256 uint4 per warp
  uint64_t* bar = reinterpret_cast<uint64_t*>(dsm + (kWarpBlock / 32) * 512) + warp * 2;
  const int64_t nwarps = (int64_t)gridDim.x * (kWarpBlock / 32);
  int64_t a = (int64_t)blockIdx.x * (kWarpBlock / 32) + warp;
  const uint32_t bytes = (uint32_t)n * 4u;
  const int nc = n >> 2;
  if (lane == 0) {
    mbar_init(&bar[0], 1);
    mbar_init(&bar[1], 1);
    fence_mbar_init();
    if (a < N) {
      mbar_arrive_expect_tx(&bar[0], bytes);
      bulk_g2s(buf0, d + a * (int64_t)n, bytes, &bar[0]);
    }
  }
  __syncwarp();
  for (uint32_t t = 0; a < N; ++t, a += nwarps) {
    const uint32_t b = t & 1u;
    uint4* cur = buf0 + b * 256;
    const int64_t an = a + nwarps;
    if (lane == 0 && an < N) {  // prefetch the next array into the other buffer
      mbar_arrive_expect_tx(&bar[b ^ 1u], bytes);
      bulk_g2s(buf0 + (b ^ 1u) * 256, d + an * (int64_t)n, bytes, &bar[b ^ 1u]);
    }
    mbar_wait_parity(&bar[b], (t >> 1) & 1u);
    uint32_t k[32];
#pragma unroll
    for (int q = 0; q < 8; ++q) {
      const int c = lane + 32 * q;
      uint4 v = make_uint4(kPadKey, kPadKey, kPadKey, kPadKey);
      if (c < nc) {
        v = cur[c];
        v.x = key_from_bits(v.x); v.y = key_from_bits(v.y);
        v.z = key_from_bits(v.z); v.w = key_from_bits(v.w);
      }
      k[4 * q + 0] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
    }
    __syncwarp();  // every lane has its data: the buffer becomes sort scratch
    sort1024_warp(k, lane, reinterpret_cast<uint32_t*>(cur), one);
    stage_out<32>(k, cur, lane * 8);
    __syncwarp();
    uint4* dst = reinterpret_cast<uint4*>(d + a * (int64_t)n);
#pragma unroll
    for (int q = 0; q < 8; ++q) {
      const int c = lane + 32 * q;
      if (c < nc) st_stream(dst + c, cur[swz(c)]);
    }
    fence_proxy_async_smem();  // generic reads of `cur` before the next bulk write into it
    __syncwarp();
  }
}

#ifndef GAS_CTA_WARPS_PER_SM
#define GAS_CTA_WARPS_PER_SM 20  // occupancy target (measured: 20 > 16, 24, 12) of the CTA classes (register budget 65536 / (32 x this))
#endif

template <int W, int WR>
constexpr int cta_smem_bytes() { return 1024 * W * 4 + WR * 4096; }

// CTA-level classes: P = 1024 * W (W = 2, 4, 8, 16), one array per CTA of 32*WR
// threads (WR <= W real warps: n <= 1024 * WR, see sort_cta).
template <int W, int WR, bool VEC>
__global__ void __launch_bounds__(32 * WR, (GAS_CTA_WARPS_PER_SM / WR > 0 ? GAS_CTA_WARPS_PER_SM / WR : 1)) k_fixed_cta(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one) {
  constexpr int KPT = 32, T = 32 * WR, P = KPT * 32 * W;
  // dynamic shared memory (cta_smem_bytes<W, WR>()): P words of cross-warp
  // exchange / rank-order staging, then a 4 KB transpose scratch per warp
  extern __shared__ __align__(16) uint4 cta_smem[];
  uint4* smem = cta_smem;
  uint32_t* xs = reinterpret_cast<uint32_t*>(smem);
  const int t = threadIdx.x, lane = t & 31;
  uint32_t* wbuf = reinterpret_cast<uint32_t*>(cta_smem + P / 4 + (t >> 5) * 256);
  for (int64_t a = blockIdx.x; a < N; a += gridDim.x) {
    uint32_t k[KPT];
    load_keys<KPT, T, VEC>(k, d + a * (int64_t)n, n, t, true);
    fill_virtual<W, WR>(xs, t);
    sort_cta<W>(k, t, lane, xs, wbuf, one);
    __syncthreads();
    stage_out_words<KPT>(k, smem, t * KPT);
    __syncthreads();
    if constexpr (VEC) {
      const int nc = n >> 2;
#pragma unroll
      for (int q = 0; q < KPT / 4; ++q) {
        const int c = t + T * q;
        if (c < nc) st_stream(reinterpret_cast<uint4*>(d + a * (int64_t)n) + c, smem[swz(c)]);
      }
    } else {
#pragma unroll
      for (int q = 0; q < KPT; ++q) {
        const int w = t + T * q;
        if (w < n) st_stream(d + a * (int64_t)n + w, sword(smem, w));
      }
    }
    __syncthreads();
  }
}

// ===================================================== variable-length kernels
// Array i = d[off[i] .. off[i+1]). A launch handles the arrays of one size
// class (len in (P/2, P], or len == 2 for P == 2). Warps scan windows of 32
// arrays, ballot the in-class ones and sort them GROUPS at a time, so that
// no device workspace (index lists) is needed. Offsets may have any 4-byte
// alignment, so loads/stores are scalar and masked to [off[i], off[i+1]).

__device__ __forceinline__ bool in_class(int64_t len, int P) {
  return P == 2 ? len == 2 : (len > P / 2 && len <= P);
}

template <int KPT, int G>
__global__ void __launch_bounds__(warp_block<G>(), warp_block_min<G>()) k_offsets_warp(uint32_t* __restrict__ d, const int64_t* __restrict__ off,
                                                          int64_t N, uint32_t one) {
  constexpr int GROUPS = 32 / G;
  constexpr int P = KPT * G;
  constexpr int BLK = warp_block<G>();
  extern __shared__ uint4 warp_dsm[];  // warp_smem_bytes<KPT, G>()
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const int g = lane & (G - 1), grp = lane / G;
  uint4* sb = warp_dsm + warp * warp_smem_chunks<KPT>();
  const int64_t nwarps = (int64_t)gridDim.x * (BLK / 32);
  for (int64_t win = ((int64_t)blockIdx.x * (BLK / 32) + warp) * 32; win < N; win += nwarps * 32) {
    const int64_t mine = win + lane;
    int64_t my_lo = 0, my_len = 0;
    if (mine < N) { my_lo = off[mine]; my_len = off[mine + 1] - my_lo; }
    uint32_t mask = __ballot_sync(0xffffffffu, mine < N && in_class(my_len, P));
    while (mask) {
      const int cnt = __popc(mask);
      const bool valid = grp < cnt;
      const int pos = valid ? (int)__fns(mask, 0, grp + 1) : 0;
      const int64_t lo = __shfl_sync(0xffffffffu, my_lo, pos);
      const int len = (int)__shfl_sync(0xffffffffu, my_len, pos);
      // the other groups' slots of this round, for the store phase
      uint32_t k[KPT];
      load_keys<KPT, G, false>(k, d + lo, len, g, valid);
      if constexpr (KPT == 32 && G >= 2) sort_group_warp<G>(k, g, reinterpret_cast<uint32_t*>(sb), one);
      else Bitonic<KPT, G, 1>::sort(k, g, 0, nullptr, one);
      stage_out_words<KPT>(k, sb, grp * P + g * KPT);
      __syncwarp();
#pragma unroll
      for (int q = 0; q < KPT; ++q) {
        const int w = lane + 32 * q;
        const int gg = w / P, pw = w % P;
        const int64_t glo = __shfl_sync(0xffffffffu, lo, gg * G);
        const int glen = __shfl_sync(0xffffffffu, valid ? len : 0, gg * G);
        if (pw < glen) st_stream(d + glo + pw, sword(sb, w));
      }
      __syncwarp();
      if (cnt <= GROUPS) {
        mask = 0;
      } else {
        const int last = (int)__fns(mask, 0, GROUPS);
        mask &= (last >= 31) ? 0u : (0xffffffffu << (last + 1));
      }
    }
  }
}

template <int W, int WR>
__global__ void __launch_bounds__(32 * WR, (GAS_CTA_WARPS_PER_SM / WR > 0 ? GAS_CTA_WARPS_PER_SM / WR : 1)) k_offsets_cta(uint32_t* __restrict__ d, const int64_t* __restrict__ off,
                                                         int64_t N, int64_t LO, int64_t HI,
                                                         unsigned long long* __restrict__ ctr, uint32_t one) {
  // handles the arrays with LO < length <= HI (HI <= 1024 * WR)
  constexpr int KPT = 32, T = 32 * WR, P = KPT * 32 * W;
  extern __shared__ __align__(16) uint4 cta_smem[];
  uint4* smem = cta_smem;
  uint32_t* xs = reinterpret_cast<uint32_t*>(smem);
  const int t = threadIdx.x, g = t & 31;
  uint32_t* wbuf = reinterpret_cast<uint32_t*>(cta_smem + P / 4 + (t >> 5) * 256);
  // windows of 32 arrays are handed out dynamically through `ctr` (one counter
  // per launch, zeroed by the host) so that CTAs finish together even though
  // the number of in-class arrays per window varies
  __shared__ int64_t s_win;
  auto next_window = [&]() -> int64_t {
    if (t == 0) s_win = (int64_t)atomicAdd(ctr, 1ull) * 32;
    __syncthreads();
    const int64_t w = s_win;
    __syncthreads();
    return w;
  };
  for (int64_t win = next_window(); win < N; win = next_window()) {
    const int64_t mine = win + g;
    int64_t my_lo = 0, my_len = 0;
    if (mine < N) { my_lo = off[mine]; my_len = off[mine + 1] - my_lo; }
    uint32_t mask = __ballot_sync(0xffffffffu, mine < N && my_len > LO && my_len <= HI);
    while (mask) {  // identical in every warp of the CTA
      const int pos = __ffs(mask) - 1;
      mask &= mask - 1;
      const int64_t lo = __shfl_sync(0xffffffffu, my_lo, pos);
      const int len = (int)__shfl_sync(0xffffffffu, my_len, pos);
      uint32_t k[KPT];
      load_keys<KPT, T, false>(k, d + lo, len, t, true);
      fill_virtual<W, WR>(xs, t);
      sort_cta<W>(k, t, g, xs, wbuf, one);
      __syncthreads();
      stage_out_words<KPT>(k, smem, t * KPT);
      __syncthreads();
#pragma unroll
      for (int q = 0; q < KPT; ++q) {
        const int w = t + T * q;
        if (w < len) st_stream(d + lo + w, sword(smem, w));
      }
      __syncthreads();
    }
  }
}

}  // namespace gas
