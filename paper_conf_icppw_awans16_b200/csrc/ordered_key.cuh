// ordered_key.cuh — float32 bit pattern <-> order-preserving uint32 key.
//
// DESIGN.md reading C-1: the "<=" of PAPER.md Definition 1 is
// IEEE 754-2008 §5.10 totalOrder. On binary32 it is exactly unsigned order of
//     key(u) = u ^ (sign(u) ? 0xFFFFFFFF : 0x80000000)
// (negatives: all bits flipped, so larger magnitude -> smaller key and
//  -NaN < -inf; positives: sign bit set, so every positive > every negative).
// Checked over all 2^32 patterns, through the sort kernels, by
// tests/test_ordered_key.py::test_every_bit_pattern_through_the_gpu.
//
// Sorting happens on keys only; the kernels never apply float arithmetic to
// data (no NaN quieting, no FTZ), so the output is a permutation of the input
// bit patterns.
#pragma once
#include <cstdint>

namespace gas {

// Padding for the slots n..P-1 of a size class: the maximal key. It decodes
// to 0x7FFFFFFF (+qNaN with the largest payload), which sorts after every
// other pattern; "+inf" padding would wrongly precede +NaN inputs (SURVEY §7
// hard part 2). Pads are never stored.
constexpr uint32_t kPadKey = 0xFFFFFFFFu;

__device__ __forceinline__ uint32_t key_from_bits(uint32_t u) {
  return u ^ ((uint32_t)((int32_t)u >> 31) | 0x80000000u);
}

__device__ __forceinline__ uint32_t bits_from_key(uint32_t k) {
  return k ^ (((k >> 31) - 1u) | 0x80000000u);
}

}  // namespace gas
