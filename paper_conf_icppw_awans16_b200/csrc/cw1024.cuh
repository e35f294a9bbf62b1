// cw1024.cuh — distribution-robust sort of one array of 512 < n <= 1024 keys
// by one warp: a counting sort on 2048 fine bins, then one 32-key network per
// lane over 32 consecutive positions, then a half-merge with each neighbour
// lane, then a sortedness check (kernel k_fixed_cw1024).
//
// Why: the value-bucket kernel (bucket1024.cuh) puts each key straight into a
// fixed 32-slot row of one of 64 buckets. That is fast when the values are
// flat over [min, max], as in the paper's data. Any bucket
// holding more than 32 keys, or any NaN or infinity, sends the whole array to
// the 1024-key network, which costs ~1.7x as much. Peaked values (spectra
// intensities, the paper's motivating workload), duplicate-heavy
// arrays and mixes of ±0 / inf / NaN hit that case on nearly every array.
// This kernel has no capacity limit to overflow. Its cost does not depend on
// the data, as long as no bin holding more than 9 keys holds two distinct
// keys.
//
// Per array (lane l; positions p = 0..1023, lane l's window = [32 l, 32 l + 32)):
//  1. map every key (the ordered key of ordered_key.cuh; for all-positive
//     finite arrays the raw bits, which order the same way) to a fine bin
//         f = (key - kmin) >> sh,  sh = max(0, bitlen(kmax - kmin) - 11),
//     in [0, 2047] and non-decreasing in the key. Key-linear bins follow the
//     float's binade structure, so log-normal intensities get as many bins
//     per binade as uniform data. In duplicate mode (the caller's sample saw
//     repeated values) the two low bits of f are replaced by lane & 3: each
//     bin of 4 gets 4 sub-counters, so the 32 lanes of an atomic rarely hit one
//     address (keys inside a bin are unordered anyway);
//  2. histogram: one shared-memory RED per key on 16-bit bin counters (two
//     per word; a count never exceeds 1024, so halves never carry);
//  3. exclusive scan of the 2048 counts (lane l scans bins 64 l .. 64 l + 63,
//     then a warp scan of the lane totals): counter f = first position of bin f;
//  4. scatter: an atomic add on the key's bin counter returns the key's
//     position. Keys land grouped by bin, in bin order: a key is at most
//     (its bin's count - 1) positions from its final place, and a bin holding
//     one distinct key needs no further ordering;
//  5. lane l loads its window, sorts it with the 191-comparator odd-even
//     network, and merges its 8 lowest keys with lane l-1's 8 highest and its
//     8 highest with lane l+1's 8 lowest (one max/min step plus a 3-stage
//     bitonic clean on each side: the upper / lower half of the merge). This
//     repairs every bin that straddles a window boundary with at most 8 keys
//     on each side;
//  6. check: each lane's three sorted segments join in order and lane l's
//     last key <= lane l+1's first. Sorted plus a permutation of the input
//     means correct, whatever the data. Arrays failing the check (a bin of > 9
//     keys with two distinct values) are sorted by the 1024-key network
//     (warp1024.cuh) from the same registers;
//  7. store in place (keys -> bits for non-raw arrays).
// The pieces of the paper kept: data-independent buckets whose concatenation
// is the sorted array (§4.1), bucket sizes in an array Z (Def. 4,
// P:L251-255) and bucket starts from their prefix sums. The
// paper's sample/splitter phase (Alg. 1) becomes an exact histogram over
// arithmetic fine bins, and Phase 3's per-bucket insertion sort becomes
// per-window networks.
#pragma once
#include <cstdint>

#include "segsort.cuh"
#include "bucket1024.cuh"

namespace gas {

#ifndef GAS_CW_BLOCK
#define GAS_CW_BLOCK 640
#endif
#ifndef GAS_CW_MIX_NUM  // compare-exchanges of the window network in FMA form: NUM out of DEN
#define GAS_CW_MIX_NUM 0  // all on the ALU pipe: 128 fewer instructions than 2/3 FMA form (smaller hot code), measured 1-4% faster
#endif
#ifndef GAS_CW_MIX_DEN
#define GAS_CW_MIX_DEN 3
#endif
#ifndef GAS_CW_GROUP
#define GAS_CW_GROUP 4
#endif
constexpr int kCwBlock = GAS_CW_BLOCK;
constexpr int kCwCntBytes = 4096;                   // 2048 16-bit bin counters, two per word
constexpr int kCwBufBytes = 4096;                   // 1024 positions
constexpr int kCwWarpBytes = kCwCntBytes + kCwBufBytes;
constexpr int kCwSmemBytes = (kCwBlock / 32) * kCwWarpBytes;

// Word w of a 1024-word area lives at word cw_swz(w): the 16-byte chunk
// (w >> 2) & 7 of row w >> 5 is XOR-ed with (row & 7). Lane l reading row l
// with LDS.128 (8 lanes per wavefront) and coalesced chunk reads are both
// conflict-free.
__device__ __forceinline__ uint32_t cw_swz(uint32_t w) { return w ^ ((w >> 3) & 0x1Cu); }

// (GAS_ATOM_NOPRED: unpredicated, adding 0 when !p; see atoms_add4_if in bucket1024.cuh)
__device__ __forceinline__ void reds_add_if(bool p, uint32_t a, uint32_t v) {
#if GAS_ATOM_NOPRED
  asm volatile("red.shared.add.u32 [%0], %1;" ::"r"(a), "r"(p ? v : 0u) : "memory");
#else
  asm volatile("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %0, 0;\n\t@q red.shared.add.u32 [%1], %2;\n\t}"
               ::"r"((uint32_t)p), "r"(a), "r"(v) : "memory");
#endif
}
__device__ __forceinline__ uint32_t atoms_add_if(bool p, uint32_t a, uint32_t v) {
#if GAS_ATOM_NOPRED
  uint32_t r;
  asm volatile("atom.shared.add.u32 %0, [%1], %2;" : "=r"(r) : "r"(a), "r"(p ? v : 0u) : "memory");
  return r;
#else
  uint32_t r = 0;
  asm volatile("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %1, 0;\n\t@q atom.shared.add.u32 %0, [%2], %3;\n\t}"
               : "+r"(r) : "r"((uint32_t)p), "r"(a), "r"(v) : "memory");
  return r;
#endif
}

__device__ __forceinline__ uint32_t cw_kl_shift(uint32_t kmin, uint32_t kmax) {
  const uint32_t dk = kmax - kmin;
  const int bits = 32 - __clz(dk);  // bit length of the range
  return bits > 11 ? (uint32_t)(bits - 11) : 0u;
}
// Key r of this lane lies inside the array: VEC, chunk layout (key r is
// element 4 (lane + 32 (r/4)) + r%4; n > 512 so chunks 0..3 always exist);
// scalar layout (key r is element lane + 32 r).
template <bool VEC>
__device__ __forceinline__ bool cw_valid(int r, int lane, int n) {
  return VEC ? ((r >> 2) < 4 || lane + 32 * (r >> 2) < (n >> 2)) : (r < 16 || lane + 32 * r < n);
}

// Step 5's neighbour half-merges and step 6's check. k holds the lane's sorted
// window; returns whether the warp's 1024 keys are now in order.
__device__ __forceinline__ bool cw_merge_check(uint32_t (&k)[32], int lane, uint32_t one) {
  uint32_t lo[8], hi[8];
#pragma unroll
  for (int i = 0; i < 8; ++i) {
    lo[i] = __shfl_up_sync(0xffffffffu, k[24 + i], 1);  // lane l-1's 8 highest
    hi[i] = __shfl_down_sync(0xffffffffu, k[i], 1);     // lane l+1's 8 lowest
  }
  if (lane == 0) {
#pragma unroll
    for (int i = 0; i < 8; ++i) lo[i] = 0u;
  }
  if (lane == 31) {
#pragma unroll
    for (int i = 0; i < 8; ++i) hi[i] = 0xFFFFFFFFu;
  }
  // upper half of merge(lo, k[0..7]) and lower half of merge(k[24..31], hi):
  // one max / min step makes each a bitonic 8-sequence, then clean it
#pragma unroll
  for (int i = 0; i < 8; ++i) {
    k[i] = max(k[i], lo[7 - i]);
    k[24 + i] = min(k[24 + i], hi[7 - i]);
  }
#pragma unroll
  for (int j = 4; j >= 1; j >>= 1) {
#pragma unroll
    for (int i = 0; i < 8; ++i) {
      if (!(i & j)) {
        ce_n(i, k[i], k[i | j], one);
        ce_n(i + 1, k[24 + i], k[24 + (i | j)], one);
      }
    }
  }
  const uint32_t next = __shfl_down_sync(0xffffffffu, k[0], 1);
  const bool ok = k[7] <= k[8] && k[23] <= k[24] && (lane == 31 || k[31] <= next);
  return __all_sync(0xffffffffu, ok);
}

// Steps 1-7 for one array held by the warp. k: the array's raw bits as loaded
// (VEC: chunk layout, else scalar layout; slots past the end hold a copy of
// k[0]). raw: every value positive and finite (the bits are the keys),
// umin / umax their min / max. dm: 0, or 3 for duplicate mode. cnt_sa / buf_sa:
// this warp's two 4 KB shared areas (buf_ptr = buf_sa as a pointer). Writes the
// sorted array to arr; returns true when the check failed and the network
// sorted it.
template <bool VEC>
__device__ __forceinline__ bool cw_sort_warp(uint32_t (&k)[32], bool raw, uint32_t kmin, uint32_t kmax, uint32_t dm,
                                             uint32_t* arr, int n, int lane, uint32_t cnt_sa, uint32_t buf_sa,
                                             uint32_t* buf_ptr, uint32_t one) {
  // byte offset of row `lane` in a 1024-word area, and of its chunk q (q ^ (lane & 7)).
  // Opaque moves: without them the compiler hoists the 3 x 8 chunk addresses
  // out of the caller's array loop and spills them.
  uint32_t row_sa, sw;
  asm volatile("mov.b32 %0, %1;" : "=r"(row_sa) : "r"((uint32_t)lane << 7));
  asm volatile("mov.b32 %0, %1;" : "=r"(sw) : "r"(((uint32_t)lane & 7u) << 4));
  // zero the bin counters; pad keys at positions n .. 1023
#pragma unroll
  for (int q = 0; q < 8; ++q) sts128(cnt_sa + row_sa + (((uint32_t)q << 4) ^ sw), make_uint4(0, 0, 0, 0));
  for (int p = n + lane; p < 1024; p += 32) sts32(buf_sa + cw_swz(p) * 4u, kPadKey);
  if (!raw) {
#pragma unroll
    for (int r = 0; r < 32; ++r) k[r] = key_from_bits(k[r]);
    kmin = k[0];
    kmax = k[0];
#pragma unroll
    for (int r = 1; r < 31; r += 2) {
      kmin = __vimin3_u32(kmin, k[r], k[r + 1]);
      kmax = __vimax3_u32(kmax, k[r], k[r + 1]);
    }
    kmin = __reduce_min_sync(0xffffffffu, min(kmin, k[31]));
    kmax = __reduce_max_sync(0xffffffffu, max(kmax, k[31]));
  }
  const uint32_t sh = cw_kl_shift(kmin, kmax);
  __syncwarp();
  // ---- 2. histogram (16-bit counters, two per word: a count never exceeds
  // 1024, so the halves never carry into each other). Groups of 8: the last
  // atomic of a group returns a value that is folded (AND with an opaque zero)
  // into the next group's base address, so the compiler cannot compute all 32
  // addresses up front (that spills).
  {
    const uint32_t zero = one ^ 1u;
    uint32_t kb = kmin;  // kmin, re-derived after every group from an atomic's result
#pragma unroll
    for (int r = 0; r < 32; ++r) {
      const uint32_t f = (k[r] - kb) >> sh;
      const uint32_t a = cnt_sa + cw_swz(f >> 1) * 4u, v = 1u << ((f & 1u) << 4);
      if ((r & 7) == 7) kb = kmin + (atoms_add_if(cw_valid<VEC>(r, lane, n), a, v) & zero);
      else reds_add_if(cw_valid<VEC>(r, lane, n), a, v);
    }
  }
  __syncwarp();
  // ---- 3. exclusive scan: lane l owns words 32 l .. 32 l + 31 (bins 64 l ..).
  // Word i = (count of bin 2i) | (count of bin 2i+1) << 16 becomes (start of
  // bin 2i) | (start of bin 2i+1) << 16. (Unrolled, the chunks kept in
  // registers: rolled loops that read the chunks twice measured 5-7% slower.)
  {
    uint32_t c[32];
    uint32_t tot = 0;  // packed: low half = sum of even bins, high = odd bins
#pragma unroll
    for (int q = 0; q < 8; ++q) {
      const uint4 v = lds128(cnt_sa + row_sa + (((uint32_t)q << 4) ^ sw));
      c[4 * q] = v.x; c[4 * q + 1] = v.y; c[4 * q + 2] = v.z; c[4 * q + 3] = v.w;
      tot += v.x + v.y + v.z + v.w;
    }
    const uint32_t run_lane = (tot & 0xFFFFu) + (tot >> 16);
    uint32_t x = run_lane;
#pragma unroll
    for (int s = 1; s < 32; s <<= 1) {
      const uint32_t y = __shfl_up_sync(0xffffffffu, x, s);
      if (lane >= s) x += y;
    }
    uint32_t run = x - run_lane;  // first position of this lane's bins
#pragma unroll
    for (int i = 0; i < 32; ++i) {
      const uint32_t w = c[i], t = w << 16;
      c[i] = run * 0x10001u + t;
      run += (w + t) >> 16;
    }
#pragma unroll
    for (int q = 0; q < 8; ++q)
      sts128(cnt_sa + row_sa + (((uint32_t)q << 4) ^ sw), make_uint4(c[4 * q], c[4 * q + 1], c[4 * q + 2], c[4 * q + 3]));
  }
  __syncwarp();
  // ---- 4. scatter into bin order: the atomic's old value is the position
  uint32_t kb = kmin;  // as in step 2: re-derived from each group's last atomic
#pragma unroll
  for (int g = 0; g < 32; g += GAS_CW_GROUP) {
    uint32_t old[GAS_CW_GROUP], sft[GAS_CW_GROUP];
#pragma unroll
    for (int r = g; r < g + GAS_CW_GROUP; ++r) {
      const uint32_t f = (k[r] - kb) >> sh;
      sft[r - g] = (f & 1u) << 4;
      old[r - g] = atoms_add_if(cw_valid<VEC>(r, lane, n), cnt_sa + cw_swz(f >> 1) * 4u, 1u << sft[r - g]);
    }
#pragma unroll
    for (int r = g; r < g + GAS_CW_GROUP; ++r)
      sts32_if(cw_valid<VEC>(r, lane, n), buf_sa + cw_swz((old[r - g] >> sft[r - g]) & 0xFFFFu) * 4u, k[r]);
    kb = kmin + (old[GAS_CW_GROUP - 1] & (one ^ 1u));
  }
  __syncwarp();
  // ---- 5. window network + neighbour merges, 6. check
#pragma unroll
  for (int q = 0; q < 8; ++q) {
    const uint4 v = lds128(buf_sa + row_sa + (((uint32_t)q << 4) ^ sw));
    k[4 * q] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
  }
  {  // Batcher's 32-key odd-even merge sort (191 compare-exchanges)
    constexpr OddEvenTable<32> T{};
#pragma unroll
    for (int c = 0; c < OddEvenTable<32>::C; ++c) {
      if ((c % GAS_CW_MIX_DEN) < GAS_CW_MIX_NUM) ce<true>(k[T.e[c].a], k[T.e[c].b], one);
      else ce<false>(k[T.e[c].a], k[T.e[c].b], one);
    }
  }
  const bool fell = !cw_merge_check(k, lane, one);
  if (fell) {
    __syncwarp();
    sort1024_warp(k, lane, buf_ptr, one);  // any permutation of the keys is a valid input
  }
  // ---- 7. store in place (through shared memory: coalesced)
  if (!raw) {
#pragma unroll
    for (int r = 0; r < 32; ++r) k[r] = bits_from_key(k[r]);
  }
  __syncwarp();
#pragma unroll
  for (int q = 0; q < 8; ++q)
    sts128(buf_sa + row_sa + (((uint32_t)q << 4) ^ sw), make_uint4(k[4 * q], k[4 * q + 1], k[4 * q + 2], k[4 * q + 3]));
  __syncwarp();
  if constexpr (VEC) {
    uint4* const dst = reinterpret_cast<uint4*>(arr);
    const int nc = n >> 2;
#pragma unroll
    for (int q = 0; q < 8; ++q) {
      const int c = lane + 32 * q;
      stg_cs_if(q < 4 || c < nc, dst + c, lds128(buf_sa + cw_swz(4u * c) * 4u));
    }
  } else {
#pragma unroll
    for (int r = 0; r < 32; ++r) {
      const int e = lane + 32 * r;
      if (r < 16 || e < n) st_stream(arr + e, lds32(buf_sa + cw_swz((uint32_t)e) * 4u));
    }
  }
  __syncwarp();
  return fell;
}

}  // namespace gas
