// bucket1024.cuh — bucket-then-network sort of one array of 512 < n <= 1024
// keys by one warp (the n = 1000 headline of BASELINE.json configs[1]).
//
// Why: the pure sorting network of warp1024.cuh spends ~26 compare-exchanges
// per key (levels 6-10 of a 1024-key merge network) and is bound by the
// integer-ALU pipe and instruction issue. This kernel first
// splits the array into 62 value ranges — the paper's own idea of
// data-independent buckets whose concatenation is the sorted array with no
// merge step (§4.1, Alg. 2 P:L250-297 §5.2) — and then sorts each
// bucket (<= 32 keys) with the 191-comparator odd-even network in one lane's
// registers (6 compare-exchanges per key per bucket). Differences from the
// paper, for B200: buckets come from linear interpolation between the array's
// min and max (one FADD + one FFMA per key on the FMA pipe) instead of a
// sorted sample and per-thread splitter scans (Alg. 1-2); a key's rank inside
// its bucket comes from one shared-memory atomic increment of the bucket's
// counter instead of a global bucket-size array Z (Def. 4), and
// bucket starts from a warp scan of the 62 counts; nothing but the array
// itself touches HBM.
//
// Correctness does not depend on the data: the bucket map
//     b(v) = rn(rn(v - vmin) * s + 2^23) - 2^23,   s = rn(61 / rn(vmax - vmin))
// is monotone non-decreasing in v (every step is a monotone rounding of a
// monotone function), so every key of bucket b precedes (in IEEE totalOrder,
// DESIGN.md reading C-1) every key of bucket b+1, and ±0 (equal values) share
// a bucket whose network orders them. 0 <= b <= 61 because rn(v - vmin) lies
// in [0, rn(vmax - vmin)] and range * s <= 61 (1 + 2^-24) < 61.5.
// The warp falls back to the full network (warp1024.cuh) for the whole array
// when the map cannot be used — a NaN or an infinity in the array, all values
// equal, a range that overflows or underflows — or when a bucket would hold
// more than 32 keys (measured on the paper's uniform data: 0.5% of arrays).
// The decision is warp-uniform, so both paths are branch-free inside a warp.
#pragma once
#include <cstdint>

#include "bitonic.cuh"
#include "ordered_key.cuh"
#include "warp1024.cuh"

namespace gas {

#ifndef GAS_BK_BLOCK
#define GAS_BK_BLOCK 128
#endif
#ifndef GAS_BK_WARPS_PER_SM
#define GAS_BK_WARPS_PER_SM 16
#endif
#ifndef GAS_BK_MIX_NUM  // compare-exchanges of the bucket networks in FMA form: NUM out of DEN
#define GAS_BK_MIX_NUM 2
#endif
#ifndef GAS_BK_MIX_DEN
#define GAS_BK_MIX_DEN 3
#endif
#ifndef GAS_BK_PREFETCH
#define GAS_BK_PREFETCH 1
#endif
constexpr int kBkBlock = GAS_BK_BLOCK;
// Per warp: 64 bucket counters (256 B), the slot buffer [64 buckets][36 words]
// of u32 keys (9 KB; slot p of bucket b at word 36 b + p: the 36-word stride
// makes both the random single-word scatter and the 16-byte row gathers of
// 8 consecutive lanes spread over all banks; also the 4 KB transpose scratch
// of the fallback network). Output word p is staged at word p of the slot
// buffer: rows 0..31 (1152 words >= n) are free once round 0 has gathered
// them, and round 1 reads only rows 32..63.
constexpr int kBkCntBytes = 64 * 4;
constexpr int kBkRowWords = 36;  // slot row of one bucket: 32 slots + 4 words of skew
constexpr int kBkSlotBytes = 64 * kBkRowWords * 4;
constexpr int kBkWarpBytes = kBkCntBytes + kBkSlotBytes;
constexpr int kBkSmemBytes = (kBkBlock / 32) * kBkWarpBytes;

__device__ __forceinline__ float fmin_nan(float a, float b) {
  float r;
  asm("min.NaN.f32 %0, %1, %2;" : "=f"(r) : "f"(a), "f"(b));
  return r;
}
__device__ __forceinline__ float fmax_nan(float a, float b) {
  float r;
  asm("max.NaN.f32 %0, %1, %2;" : "=f"(r) : "f"(a), "f"(b));
  return r;
}
// Shared-memory accesses as ordered (volatile) PTX; the predicated forms
// compile to one predicated instruction instead of a branch.
__device__ __forceinline__ uint32_t atoms_inc_if(bool p, uint32_t a) {
  uint32_t v = 0;
  asm volatile("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %1, 0;\n\t@q atom.shared.add.u32 %0, [%2], 1;\n\t}"
               : "+r"(v) : "r"((uint32_t)p), "r"(a) : "memory");
  return v;
}
__device__ __forceinline__ uint32_t lds32(uint32_t a) {
  uint32_t v;
  asm volatile("ld.shared.u32 %0, [%1];" : "=r"(v) : "r"(a) : "memory");
  return v;
}
__device__ __forceinline__ void sts32(uint32_t a, uint32_t v) {
  asm volatile("st.shared.u32 [%0], %1;" ::"r"(a), "r"(v) : "memory");
}
__device__ __forceinline__ void sts32_if(bool p, uint32_t a, uint32_t v) {
  asm volatile("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %0, 0;\n\t@q st.shared.u32 [%1], %2;\n\t}"
               ::"r"((uint32_t)p), "r"(a), "r"(v) : "memory");
}
__device__ __forceinline__ uint4 lds128(uint32_t a) {
  uint4 v;
  asm volatile("ld.shared.v4.u32 {%0, %1, %2, %3}, [%4];" : "=r"(v.x), "=r"(v.y), "=r"(v.z), "=r"(v.w) : "r"(a) : "memory");
  return v;
}
__device__ __forceinline__ void sts128(uint32_t a, uint4 v) {
  asm volatile("st.shared.v4.u32 [%0], {%1, %2, %3, %4};" ::"r"(a), "r"(v.x), "r"(v.y), "r"(v.z), "r"(v.w) : "memory");
}

// Bucket map of one value (see the header comment): the bits of
// rn(rn(v - vmin) * s + 2^23) are 0x4B000000 + b.
__device__ __forceinline__ uint32_t bucket_bits(uint32_t raw, float vmin, float s) {
  const float dv = __fsub_rn(__uint_as_float(raw), vmin);
  return __float_as_uint(__fmaf_rn(dv, s, 8388608.0f));
}

// Batcher's 32-input odd-even merge sort in registers with this kernel's own
// compare-exchange mix (bitonic.cuh ce<>).
__device__ __forceinline__ void sort32_bk(uint32_t (&k)[32], uint32_t one) {
  constexpr OddEvenTable<32> T{};
#pragma unroll
  for (int c = 0; c < OddEvenTable<32>::C; ++c) {
    if ((c % GAS_BK_MIX_DEN) < GAS_BK_MIX_NUM) ce<true>(k[T.e[c].a], k[T.e[c].b], one);
    else ce<false>(k[T.e[c].a], k[T.e[c].b], one);
  }
}

// The whole-array network (warp1024.cuh) for arrays the bucket map cannot
// handle. (Inline: an out-of-line call sends the key array through the stack
// on every array, measured 84 local stores per array.)
__device__ __forceinline__ void bucket1024_fallback(uint32_t (&k)[32], uint4* dst, int nc, int lane, uint32_t* scratch,
                                                    uint32_t one) {
  __syncwarp();
#pragma unroll
  for (int q = 0; q < 8; ++q) {
    const bool valid = q < 4 || lane + 32 * q < nc;
#pragma unroll
    for (int j = 0; j < 4; ++j) k[4 * q + j] = valid ? key_from_bits(k[4 * q + j]) : kPadKey;
  }
  sort1024_warp(k, lane, scratch, one);
  uint4* sb = reinterpret_cast<uint4*>(scratch);
  stage_out<32>(k, sb, lane * 8);
  __syncwarp();
#pragma unroll
  for (int q = 0; q < 8; ++q) {
    const int c = lane + 32 * q;
    if (c < nc) st_stream(dst + c, sb[swz(c)]);
  }
}

// Bucket round rho (0, 1) of one lane: gather bucket b = lane + 32 rho (its
// slot row, 8 x 16 bytes, conflict-free; slots >= size_b hold the pad key),
// sort it in registers and stage its keys at output words base_b + i, i <
// size_b. Each staging store is predicated: stores of one lane to distinct
// addresses may be reordered, so no write may rely on another lane's later
// write. RAW: keys are raw float bits (all values > 0, unsigned order = value
// order), else ordered keys (ordered_key.cuh).
template <bool RAW>
__device__ __forceinline__ void bucket_round(uint32_t (&k)[32], uint32_t row, uint32_t ob, uint32_t tb, uint32_t one) {
#pragma unroll
  for (int q = 0; q < 8; ++q) {
    const uint4 v = lds128(row + q * 16);
    k[4 * q] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
  }
  __syncwarp();  // every lane has its row before any staging store can land on rows 0..31
  sort32_bk(k, one);
#pragma unroll
  for (int i = 0; i < 32; ++i) sts32_if((uint32_t)i < tb, ob + i * 4, RAW ? k[i] : bits_from_key(k[i]));
}

// Fixed-length arrays, 512 < n <= 1024, 16-byte-aligned rows (n % 4 == 0).
// One warp per array (persistent grid-stride).
__global__ void __launch_bounds__(kBkBlock, GAS_BK_WARPS_PER_SM * 32 / kBkBlock)
    k_fixed_bucket1024(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one) {
  extern __shared__ __align__(16) uint4 bk_smem[];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const uint32_t wsa = (uint32_t)__cvta_generic_to_shared(bk_smem) + warp * kBkWarpBytes;
  const uint32_t cnt_sa = wsa;                               // counter of bucket b at cnt_sa + b*4
  const uint32_t slot_sa = wsa + kBkCntBytes;                // slot (p, b) at slot_sa + (36 b + p)*4
  const uint32_t out_sa = slot_sa;                           // output word p at out_sa + p*4 (rows 0..31)
  uint32_t* const slot_ptr = reinterpret_cast<uint32_t*>(reinterpret_cast<unsigned char*>(bk_smem) +
                                                         warp * kBkWarpBytes + kBkCntBytes);
  const int nc = n >> 2;  // 16-byte chunks per array (> 128)
  const int64_t nwarps = (int64_t)gridDim.x * (kBkBlock / 32);
  const uint32_t cnt_b0 = cnt_sa - 0x4B000000u * 4u;  // counter address = bucket bits * 4 + cnt_b0
  // slot (p, b) address = 36 * (counter address of b) + 4 p + slot_c0
  const uint32_t slot_c0 = slot_sa - (uint32_t)kBkRowWords * cnt_sa;

  for (int64_t a = (int64_t)blockIdx.x * (kBkBlock / 32) + warp; a < N; a += nwarps) {
    uint4* const dst = reinterpret_cast<uint4*>(d + a * (int64_t)n);
    // ---- a2: stage in (raw bits). Slots past the end (only in chunks q >= 4,
    // n > 512) are left out of min/max, counting and scatter.
    uint32_t k[32];
#pragma unroll
    for (int q = 0; q < 8; ++q) {
      const int c = lane + 32 * q;
      uint4 v = make_uint4(0, 0, 0, 0);
      if (q < 4 || c < nc) v = ld_stream(dst + c);
      k[4 * q] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
    }
#if GAS_BK_PREFETCH
    if (lane == 0 && a + nwarps < N)  // warm L2 with this warp's next array (one TMA bulk prefetch)
      asm volatile("cp.async.bulk.prefetch.L2.global [%0], %1;" ::"l"(d + (a + nwarps) * (int64_t)n),
                   "r"((uint32_t)n * 4u) : "memory");
#endif
    // ---- bucket map parameters: min and max value (NaN-propagating)
    float vmin = __uint_as_float(k[0]), vmax = vmin;
#pragma unroll
    for (int r = 1; r < 16; ++r) {
      vmin = fmin_nan(vmin, __uint_as_float(k[r]));
      vmax = fmax_nan(vmax, __uint_as_float(k[r]));
    }
#pragma unroll
    for (int q = 4; q < 8; ++q) {
      if (lane + 32 * q < nc) {
#pragma unroll
        for (int j = 0; j < 4; ++j) {
          vmin = fmin_nan(vmin, __uint_as_float(k[4 * q + j]));
          vmax = fmax_nan(vmax, __uint_as_float(k[4 * q + j]));
        }
      }
    }
#pragma unroll
    for (int m = 16; m >= 1; m >>= 1) {
      vmin = fmin_nan(vmin, __shfl_xor_sync(0xffffffffu, vmin, m));
      vmax = fmax_nan(vmax, __shfl_xor_sync(0xffffffffu, vmax, m));
    }
    const float range = __fsub_rn(vmax, vmin);
    const float s = __fdiv_rn(61.0f, range);
    // finite min and max (no NaN, no inf), distinct, finite range and scale
    bool use_buckets = fabsf(vmin) <= 3.402823466e38f && fabsf(vmax) <= 3.402823466e38f && range > 0.0f &&
                       range <= 3.402823466e38f && s <= 3.402823466e38f;
    // every value > 0 (no zero of either sign, no negative): raw bits sort as unsigned
    const bool raw = vmin > 0.0f;
    uint32_t t0 = 0, t1 = 0, base0 = 0, base1 = 0;
    if (use_buckets) {
      // slot buffer <- pad keys, bucket counters <- 0 (the previous array is done with both)
#pragma unroll
      for (int q = 0; q < kBkSlotBytes / 16 / 32; ++q)
        sts128(slot_sa + (lane + 32 * q) * 16, make_uint4(kPadKey, kPadKey, kPadKey, kPadKey));
      if (lane < 16) sts128(cnt_sa + lane * 16, make_uint4(0, 0, 0, 0));
      __syncwarp();
      // ---- rank: a shared-memory atomic increment of the key's bucket counter
      // returns its rank inside the bucket (any order of equal-bucket keys is
      // fine: the bucket is sorted afterwards)
      uint32_t rk[32];
#pragma unroll
      for (int r = 0; r < 32; ++r) {
        const int q = r >> 2;
        rk[r] = atoms_inc_if(q < 4 || lane + 32 * q < nc, bucket_bits(k[r], vmin, s) * 4u + cnt_b0);
      }
      __syncwarp();
      t0 = lds32(cnt_sa + lane * 4);
      t1 = lds32(cnt_sa + 128 + lane * 4);
      use_buckets = __all_sync(0xffffffffu, t0 <= 32u && t1 <= 32u);
      if (use_buckets) {
        // bucket bases: exclusive scan of the 64 bucket sizes (two 16-bit halves)
        uint32_t x = t0 | (t1 << 16);
#pragma unroll
        for (int m = 1; m < 32; m <<= 1) {
          const uint32_t y = __shfl_up_sync(0xffffffffu, x, m);
          if (lane >= m) x += y;
        }
        const uint32_t total_lo = __shfl_sync(0xffffffffu, x & 0xFFFFu, 31);
        base0 = (x & 0xFFFFu) - t0;
        base1 = total_lo + (x >> 16) - t1;
        // ---- scatter: key of rank p in bucket b -> slot (p, b), addressed
        // from the counter address ca = cnt_sa + 4 b
#pragma unroll
        for (int r = 0; r < 32; ++r) {
          const int q = r >> 2;
          const uint32_t ca = bucket_bits(k[r], vmin, s) * 4u + cnt_b0;
          const uint32_t sa = ca * (uint32_t)kBkRowWords + (rk[r] * 4u + slot_c0);
          sts32_if(q < 4 || lane + 32 * q < nc, sa, raw ? k[r] : key_from_bits(k[r]));
        }
        __syncwarp();
      }
    }

    if (use_buckets) {
      // ---- two bucket rounds per lane (rolled: the hot code stays in the
      // instruction cache), then the coalesced in-place store
      if (raw) {
#pragma unroll 1
        for (int rho = 0; rho < 2; ++rho)
          bucket_round<true>(k, slot_sa + (lane + 32 * rho) * (kBkRowWords * 4), out_sa + (rho ? base1 : base0) * 4, rho ? t1 : t0,
                             one);
      } else {
#pragma unroll 1
        for (int rho = 0; rho < 2; ++rho)
          bucket_round<false>(k, slot_sa + (lane + 32 * rho) * (kBkRowWords * 4), out_sa + (rho ? base1 : base0) * 4, rho ? t1 : t0,
                              one);
      }
      __syncwarp();
#pragma unroll
      for (int q = 0; q < 8; ++q) {
        const int c = lane + 32 * q;
        if (c < nc) st_stream(dst + c, lds128(out_sa + c * 16));
      }
    } else {
      bucket1024_fallback(k, dst, nc, lane, slot_ptr, one);
    }
    __syncwarp();
  }
}

}  // namespace gas
