// warp1024.cuh — specialised sort of one 1024-key segment by one warp
// (size class P = 1024, the n = 1000 headline of BASELINE.json configs[1]).
//
// Same network family as bitonic.cuh (mirror-form bitonic merges, every
// compare-exchange ascending), re-organised for the B200 instruction budget
// measured in tools/microbench.cu (VIMNMX and IMAD 64/clk/SM each, SHFL
// 32/clk/SM, issue 128/clk/SM):
//   levels 1-5   Batcher odd-even merge sort of the thread's 32 registers
//                (191 compare-exchanges instead of bitonic's 240);
//   levels 6-10  one rolled loop (keeps the hot code inside the instruction
//                cache): the mirror stage over lanes with SHFL.BFLY, then
//                the cleaners at lane distances — as SHFL stages for levels
//                6-7, and for levels 8-10 after a 32x32 transpose through
//                shared memory, as in-register stages — then a transpose
//                back and the five in-register cleaners.
// Layout A (default): element i = lane*32 + r is register r of lane `lane`.
// Layout B (after transpose): element i = r*32 + lane.
#pragma once
#include <cstdint>

#include "bitonic.cuh"

namespace gas {

// ---- Batcher odd-even merge sort network on 32 inputs, as a constexpr table.
struct CePair { int a, b; };

template <int N>
struct OddEvenTable {
  static constexpr int count() {
    int c = 0;
    for (int p = 1; p < N; p <<= 1)
      for (int k = p; k >= 1; k >>= 1)
        for (int j = k % p; j + k < N; j += 2 * k)
          for (int i = 0; i < (k < N - j - k ? k : N - j - k); ++i)
            if ((i + j) / (2 * p) == (i + j + k) / (2 * p)) ++c;
    return c;
  }
  static constexpr int C = count();
  CePair e[C];
  constexpr OddEvenTable() : e() {
    int c = 0;
    for (int p = 1; p < N; p <<= 1)
      for (int k = p; k >= 1; k >>= 1)
        for (int j = k % p; j + k < N; j += 2 * k)
          for (int i = 0; i < (k < N - j - k ? k : N - j - k); ++i)
            if ((i + j) / (2 * p) == (i + j + k) / (2 * p)) e[c++] = CePair{i + j, i + j + k};
  }
};

__device__ __forceinline__ void sort32_regs(uint32_t (&k)[32], uint32_t one) {
  constexpr OddEvenTable<32> T{};
  static_assert(OddEvenTable<32>::C == 191, "Batcher odd-even merge sort of 32 has 191 comparators");
#pragma unroll
  for (int c = 0; c < OddEvenTable<32>::C; ++c) ce_n(c, k[T.e[c].a], k[T.e[c].b], one);
}

// In-register cleaners at register distances 16, 8, 4, 2, 1 (a bitonic
// half-cleaner cascade: sorts a bitonic sequence held in 32 registers).
__device__ __forceinline__ void cleaners32(uint32_t (&k)[32], uint32_t one) {
  Bitonic<32, 1, 1>::reg_stage<16>(k, one);
  Bitonic<32, 1, 1>::reg_stage<8>(k, one);
  Bitonic<32, 1, 1>::reg_stage<4>(k, one);
  Bitonic<32, 1, 1>::reg_stage<2>(k, one);
  Bitonic<32, 1, 1>::reg_stage<1>(k, one);
}

// 32x32 transposes through the warp's 4 KB shared buffer `sm` (1024 words).
// A -> B: lane l writes its row (8 x STS.128, chunk-swizzled), then reads
// column l (32 x LDS.32). B -> A: the reverse. Both conflict-free.
__device__ __forceinline__ int swz_word(int row, int col) {  // word (row, col) of a 32x32 tile
  return row * 32 + ((((col >> 2) ^ (row & 7)) << 2) | (col & 3));
}

__device__ __forceinline__ void transpose_ab(uint32_t (&k)[32], uint32_t* sm, int lane) {
  uint4* s4 = reinterpret_cast<uint4*>(sm);
#pragma unroll
  for (int q = 0; q < 8; ++q) s4[lane * 8 + (q ^ (lane & 7))] = make_uint4(k[4 * q], k[4 * q + 1], k[4 * q + 2], k[4 * q + 3]);
  __syncwarp();
#pragma unroll
  for (int r = 0; r < 32; ++r) k[r] = sm[swz_word(r, lane)];
  __syncwarp();
}

__device__ __forceinline__ void transpose_ba(uint32_t (&k)[32], uint32_t* sm, int lane) {
#pragma unroll
  for (int r = 0; r < 32; ++r) sm[swz_word(r, lane)] = k[r];
  __syncwarp();
  const uint4* s4 = reinterpret_cast<const uint4*>(sm);
#pragma unroll
  for (int q = 0; q < 8; ++q) {
    const uint4 v = s4[lane * 8 + (q ^ (lane & 7))];
    k[4 * q] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
  }
  __syncwarp();
}

// Mirror stage of merge size 2^lk across lanes (lk = 6..10): partner element
// i ^ (2^lk - 1) = lane ^ m, register 31 - r.
__device__ __forceinline__ void shfl_mirror(uint32_t (&k)[32], int m, bool upper) {
#pragma unroll
  for (int r = 0; r < 16; ++r) {
    const uint32_t v1 = __shfl_xor_sync(0xffffffffu, k[31 - r], m);
    const uint32_t v2 = __shfl_xor_sync(0xffffffffu, k[r], m);
    k[r] = keep(k[r], v1, upper);
    k[31 - r] = keep(k[31 - r], v2, upper);
  }
}

__device__ __forceinline__ void shfl_cleaner(uint32_t (&k)[32], int m, bool upper) {
#pragma unroll
  for (int r = 0; r < 32; ++r) k[r] = keep(k[r], __shfl_xor_sync(0xffffffffu, k[r], m), upper);
}

#ifndef GAS_LEVEL_UNROLL
#define GAS_LEVEL_UNROLL 1  // 1: rolled level loop (instruction-cache friendly)
#endif
constexpr int kLevelUnroll = GAS_LEVEL_UNROLL;

// Sort P = 32*G keys held by a group of G lanes (32 per lane, layout A in and
// out; G in {2, ..., 32}, groups aligned inside the warp). Levels 6 ..
// 5+log2(G) run in one rolled loop; for G = 32 the lane-distance cleaners of
// levels 8-10 go through a transpose (`sm`: the warp's 1024-word buffer),
// otherwise they are SHFL stages.
template <int G>
__device__ __forceinline__ void level_step(uint32_t (&k)[32], int g, uint32_t* sm, uint32_t one, int lk) {
  shfl_mirror(k, (1 << (lk - 5)) - 1, g & (1 << (lk - 6)));
  if (lk == 7) {
    shfl_cleaner(k, 1, g & 1);
  } else if (G == 32 && lk >= 8) {
    transpose_ab(k, sm, g);  // element i = r*32 + lane: lane bits became register bits
    if (lk == 10) Bitonic<32, 1, 1>::reg_stage<8>(k, one);
    if (lk >= 9) Bitonic<32, 1, 1>::reg_stage<4>(k, one);
    Bitonic<32, 1, 1>::reg_stage<2>(k, one);
    Bitonic<32, 1, 1>::reg_stage<1>(k, one);
    transpose_ba(k, sm, g);
  } else if (lk >= 8) {
#pragma unroll 1
    for (int m = 1 << (lk - 7); m >= 1; m >>= 1) shfl_cleaner(k, m, g & m);
  }
  cleaners32(k, one);
}

#ifndef GAS_UNROLLED_LOW_LEVELS
#define GAS_UNROLLED_LOW_LEVELS 0  // levels 6..5+this are unrolled, the rest rolled
#endif

template <int G>
__device__ __forceinline__ void sort_group_warp(uint32_t (&k)[32], int g, uint32_t* sm, uint32_t one) {
  constexpr int LOGG = Log2<G>::value;
  constexpr int TOP = 5 + LOGG;
  constexpr int UNR = GAS_UNROLLED_LOW_LEVELS < LOGG ? GAS_UNROLLED_LOW_LEVELS : LOGG;
  sort32_regs(k, one);
#pragma unroll
  for (int lk = 6; lk < 6 + UNR; ++lk) level_step<G>(k, g, sm, one, lk);
#pragma unroll kLevelUnroll
  for (int lk = 6 + UNR; lk <= TOP; ++lk) level_step<G>(k, g, sm, one, lk);
}

__device__ __forceinline__ void sort1024_warp(uint32_t (&k)[32], int lane, uint32_t* sm, uint32_t one) {
  sort_group_warp<32>(k, lane, sm, one);
}

// Sort a bitonic 1024-sequence held by the warp (layout A): the half-cleaner
// cascade at distances 512 .. 1 (lane distances via a transpose to layout B).
__device__ __forceinline__ void cleaners1024_warp(uint32_t (&k)[32], int lane, uint32_t* sm, uint32_t one) {
  transpose_ab(k, sm, lane);
  cleaners32(k, one);  // element distances 512 .. 32 are register distances 16 .. 1 in layout B
  transpose_ba(k, sm, lane);
  cleaners32(k, one);
}

// One array of P = 1024 * W keys owned by a CTA of W warps (t = w*32 + lane):
// each warp sorts its 1024-block with sort1024_warp, then the merge levels
// 11 .. log2(P) run their cross-warp stages through shared memory (`xs`, P
// words, element (t, r) at xs[r*32W + t]) and finish inside each warp.
// A CTA may run with fewer real warps than W (lengths <= 1024 * real warps):
// the missing warps' blocks are all padding, their xs slots hold kPadKey
// (fill_virtual), and since they are the highest blocks every real element
// is the lower partner of a padding element, keeps its own value, and the
// network result for the real elements is unchanged.
template <int W>
__device__ __forceinline__ void sort_cta(uint32_t (&k)[32], int t, int lane, uint32_t* xs, uint32_t* wbuf,
                                         uint32_t one, uint32_t bar = 0) {
  using B = Bitonic<32, 32, W>;
  sort1024_warp(k, lane, wbuf, one);
#pragma unroll 1
  for (int lk = 11; lk <= B::LOGP; ++lk) {
    const int K = 1 << lk;
    B::smem_stage(k, xs, t, (K - 1) >> 5, 31, t & ((K >> 1) >> 5), bar);  // mirror, across warps
    for (int j = K >> 2; j >= 1024; j >>= 1) B::smem_stage(k, xs, t, j >> 5, 0, t & (j >> 5), bar);
    cleaners1024_warp(k, lane, wbuf, one);
  }
}

template <int W, int WR>
__device__ __forceinline__ void fill_virtual(uint32_t* xs, int t) {
  if constexpr (WR < W) {
    constexpr int VT = 32 * (W - WR);  // virtual threads
    for (int i = t; i < 32 * VT; i += 32 * WR) xs[(i / VT) * (32 * W) + 32 * WR + i % VT] = 0xFFFFFFFFu;
  }
}

}  // namespace gas
