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

// Sort 1024 keys held by the warp (32 per lane, layout A in and out).
// `sm` is the warp's 1024-word shared buffer.
__device__ __forceinline__ void sort1024_warp(uint32_t (&k)[32], int lane, uint32_t* sm, uint32_t one) {
  sort32_regs(k, one);
#pragma unroll kLevelUnroll
  for (int lk = 6; lk <= 10; ++lk) {
    shfl_mirror(k, (1 << (lk - 5)) - 1, lane & (1 << (lk - 6)));
    if (lk == 7) {
      shfl_cleaner(k, 1, lane & 1);
    } else if (lk >= 8) {
      transpose_ab(k, sm, lane);  // element i = r*32 + lane: lane bits became register bits
      if (lk == 10) Bitonic<32, 1, 1>::reg_stage<8>(k, one);
      if (lk >= 9) Bitonic<32, 1, 1>::reg_stage<4>(k, one);
      Bitonic<32, 1, 1>::reg_stage<2>(k, one);
      Bitonic<32, 1, 1>::reg_stage<1>(k, one);
      transpose_ba(k, sm, lane);
    }
    cleaners32(k, one);
  }
}

}  // namespace gas
