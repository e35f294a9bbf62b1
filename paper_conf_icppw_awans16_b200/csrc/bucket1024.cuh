// bucket1024.cuh — bucket-then-network sort of one array of 512 < n <= 1024
// keys by one warp (the n = 1000 headline of BASELINE.json configs[1]).
//
// Why: the pure sorting network of warp1024.cuh spends ~26 compare-exchanges
// per key (levels 6-10 of a 1024-key merge network) and is bound by the
// integer-ALU pipe and instruction issue. This kernel first
// splits the array into 64 value ranges — the paper's own idea of
// data-independent buckets whose concatenation is the sorted array with no
// merge step (§4.1, Alg. 2 P:L250-297 §5.2) — and then sorts each
// bucket (<= 32 keys) with the 191-comparator odd-even network in one lane's
// registers (6 compare-exchanges per key per bucket). Differences from the
// paper, for B200: buckets come from linear interpolation between the array's
// min and max (one FADD + one FFMA per key on the FMA pipe) instead of a
// sorted sample and per-thread splitter scans (Alg. 1-2); a key's rank inside
// its bucket comes from one shared-memory atomic increment of the bucket's
// counter instead of a global bucket-size array Z (Def. 4), and
// bucket starts from a warp scan of the 64 counts; nothing but the array
// itself touches HBM.
//
// Correctness does not depend on the data: the bucket map
//     b(v) = rn(rn(v - vmin) * s + 2^23) - 2^23,   s = rn(TOP / rn(vmax - vmin))
// is monotone non-decreasing in v (every step is a monotone rounding of a
// monotone function), so every key of bucket b precedes (in IEEE totalOrder,
// DESIGN.md reading C-1) every key of bucket b+1, and ±0 (equal values) share
// a bucket whose network orders them. 0 <= b <= TOP because rn(v - vmin) lies
// in [0, rn(vmax - vmin)] and range * s <= TOP (1 + 2^-24) < TOP + 1/2
// (TOP = GAS_BK_TOP = 63 for the warp kernel: 64 buckets; 61 W in bucket_cta.cuh).
// The warp falls back to the full network (warp1024.cuh) for the whole array
// when the map cannot be used — a NaN or an infinity in the array, all values
// equal, a range that overflows or underflows — or when a bucket would hold
// more than 32 keys (measured on the paper's uniform data: 0.5% of arrays).
// The decision is warp-uniform, so both paths are branch-free inside a warp.
#pragma once
#include <cstdint>

#include "bitonic.cuh"
#include "bulk.cuh"
#include "ordered_key.cuh"
#include "warp1024.cuh"

namespace gas {

#ifndef GAS_ATOM_NOPRED  // shared atomics without predicates (see atoms_add4_if)
#define GAS_ATOM_NOPRED 1
#endif
#ifndef GAS_BK_BLOCK
#define GAS_BK_BLOCK 768  // one block of 24 warps per SM (80 registers): 4.22 ms; 20 warps as 640 / 320 / 160 / 128-thread blocks: 4.25 / 4.33 / 4.38 / 4.39 ms
#endif
#ifndef GAS_BK_WARPS_PER_SM
#define GAS_BK_WARPS_PER_SM 24
#endif
#ifndef GAS_BK_MIX_NUM  // compare-exchanges of the bucket networks in FMA form: NUM out of DEN
#define GAS_BK_MIX_NUM 2
#endif
#ifndef GAS_BK_MIX_DEN
#define GAS_BK_MIX_DEN 3
#endif
#ifndef GAS_BK_TOP  // the fixed-length warp kernel's buckets are 0 .. GAS_BK_TOP (<= 63)
#define GAS_BK_TOP 63
#endif
#ifndef GAS_BK_TIERS  // network sizes per bucket round: 1 = always 32; 2 = 28 or 32; 3 = 24, 28 or 32
#define GAS_BK_TIERS 1
#endif
#ifndef GAS_BK_GROUP  // keys whose atomics are issued back to back before their scatter stores
#define GAS_BK_GROUP 4
#endif
#ifndef GAS_BK_TMA_STORE  // 1: the staged sorted array leaves through one TMA bulk store (cp.async.bulk) instead of 8 LDS.128 + STG.128 per lane
#define GAS_BK_TMA_STORE 1
#endif
#ifndef GAS_BK_PREFETCH  // L2 prefetch of the array this warp sorts GAS_BK_PREFETCH iterations ahead (0 = off)
#define GAS_BK_PREFETCH 1
#endif
constexpr int kBkBlock = GAS_BK_BLOCK;
// Per warp: 64 bucket counters (256 B) and the slot buffer [64 buckets][36
// words] of u32 keys (9 KB; slot p of bucket b at word 36 b + p: the 36-word
// stride makes both the random single-word scatter and the 16-byte row gathers
// of 8 consecutive lanes spread over all banks; also the 4 KB transpose
// scratch of the fallback network). Output word p is staged at slot word
// 1152 + p (rows 32..63): the first round sorts buckets 32..63, so those rows
// are drained before any output is staged, and rows 0..31 stay intact for the
// second round.
constexpr int kBkCntBytes = 64 * 4;
constexpr int kBkRowWords = 36;  // slot row of one bucket: 32 slots + 4 words of skew
constexpr int kBkSlotBytes = 64 * kBkRowWords * 4;
constexpr int kBkStageWord = 32 * kBkRowWords;  // output word p at slot word kBkStageWord + p (n <= 1152)
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
__device__ __forceinline__ uint32_t atoms_inc_pred(bool p, uint32_t a) {
  uint32_t v = 0;
  asm volatile("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %1, 0;\n\t@q atom.shared.add.u32 %0, [%2], 1;\n\t}"
               : "+r"(v) : "r"((uint32_t)p), "r"(a) : "memory");
  return v;
}
__device__ __forceinline__ uint32_t atoms_inc_if(bool p, uint32_t a) {  // see atoms_add4_if
#if GAS_ATOM_NOPRED
  uint32_t v;
  asm volatile("atom.shared.add.u32 %0, [%1], %2;" : "=r"(v) : "r"(a), "r"(p ? 1u : 0u) : "memory");
  return v;
#else
  uint32_t v = 0;
  asm volatile("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %1, 0;\n\t@q atom.shared.add.u32 %0, [%2], 1;\n\t}"
               : "+r"(v) : "r"((uint32_t)p), "r"(a) : "memory");
  return v;
#endif
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
// Stores the first tb (<= 32) registers of k at consecutive words from word
// index w0 of the shared array `sw`. The predicates are the bits of a mask, so
// ptxas sets them 7 at a time with R2P instead of 32 ISETP (GAS_BK_MASKSTORE;
// plain C++ stores: ordered against the asm shared accesses by their memory
// clobbers). XF: store bits_from_key of the keys.
#ifndef GAS_BK_MASKSTORE
#define GAS_BK_MASKSTORE 1
#endif
template <bool XF = false>
__device__ __forceinline__ void stage_first(uint32_t* sw, uint32_t w0, uint32_t tb, const uint32_t (&k)[32]);

__device__ __forceinline__ uint4 lds128(uint32_t a) {
  uint4 v;
  asm volatile("ld.shared.v4.u32 {%0, %1, %2, %3}, [%4];" : "=r"(v.x), "=r"(v.y), "=r"(v.z), "=r"(v.w) : "r"(a) : "memory");
  return v;
}
__device__ __forceinline__ void sts128(uint32_t a, uint4 v) {
  asm volatile("st.shared.v4.u32 [%0], {%1, %2, %3, %4};" ::"r"(a), "r"(v.x), "r"(v.y), "r"(v.z), "r"(v.w) : "memory");
}

template <bool XF>
__device__ __forceinline__ void stage_first(uint32_t* sw, uint32_t w0, uint32_t tb, const uint32_t (&k)[32]) {
  const uint32_t pm = tb >= 32u ? 0xFFFFFFFFu : ((1u << tb) - 1u);
#pragma unroll
  for (int i = 0; i < 32; ++i)
    if (pm & (1u << i)) sw[w0 + i] = XF ? bits_from_key(k[i]) : k[i];
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

// Batcher's odd-even merge sort of the first NK registers (NK = 24, 28, 32;
// checked exhaustively with the 0-1 principle). When registers NK..31 hold
// keys that follow every key in 0..NK-1, the first NK outputs are sorted.
template <int NK>
__device__ __forceinline__ void sortn_bk(uint32_t (&k)[32], uint32_t one) {
  constexpr OddEvenTable<NK> T{};
#pragma unroll
  for (int c = 0; c < OddEvenTable<NK>::C; ++c) {
    if ((c % GAS_BK_MIX_DEN) < GAS_BK_MIX_NUM) ce<true>(k[T.e[c].a], k[T.e[c].b], one);
    else ce<false>(k[T.e[c].a], k[T.e[c].b], one);
  }
}

// The whole-array network (warp1024.cuh) for arrays the bucket map cannot
// handle. (Inline: an out-of-line call sends the key array through the stack
// on every array, measured 84 local stores per array.)
// QV: chunks q < QV are always inside the array (n > 128 QV).
template <int QV = 4>
__device__ __forceinline__ void bucket1024_fallback(uint32_t (&k)[32], uint4* dst, int nc, int lane, uint32_t* scratch,
                                                    uint32_t one) {
  __syncwarp();
#pragma unroll
  for (int q = 0; q < 8; ++q) {
    const bool valid = q < QV || lane + 32 * q < nc;
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


// any 4-byte alignment: key r of the lane is element lane + 32 r (n > 512)
__device__ __forceinline__ void bucket1024_fallback_scalar(uint32_t (&k)[32], uint32_t* arr, int n, int lane,
                                                           uint32_t* scratch, uint32_t one) {
  __syncwarp();
#pragma unroll
  for (int r = 0; r < 32; ++r) k[r] = (r < 16 || lane + 32 * r < n) ? key_from_bits(k[r]) : kPadKey;
  sort1024_warp(k, lane, scratch, one);
  uint4* sb = reinterpret_cast<uint4*>(scratch);
  stage_out<32>(k, sb, lane * 8);
  __syncwarp();
#pragma unroll
  for (int r = 0; r < 32; ++r) {
    const int e = lane + 32 * r;
    if (e < n) st_stream(arr + e, sword(sb, e));
  }
}

// One TMA bulk prefetch into L2 of the 16-byte-aligned cover of [p, p + words).
__device__ __forceinline__ void prefetch_l2(const uint32_t* p, int64_t words) {
  const uintptr_t a = reinterpret_cast<uintptr_t>(p) & ~(uintptr_t)15;
  const uintptr_t e = (reinterpret_cast<uintptr_t>(p + words) + 15) & ~(uintptr_t)15;
  asm volatile("cp.async.bulk.prefetch.L2.global [%0], %1;" ::"l"(a), "r"((uint32_t)(e - a)) : "memory");
}


// Predicated forms of the global / shared accesses of the kernel below (one
// predicated instruction each instead of a branch around it).
__device__ __forceinline__ uint4 ldg_cs_if(bool p, const uint4* a) {
  uint4 v = make_uint4(0, 0, 0, 0);
  asm volatile("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %4, 0;\n\t@q ld.global.cs.v4.u32 {%0, %1, %2, %3}, [%5];\n\t}"
               : "+r"(v.x), "+r"(v.y), "+r"(v.z), "+r"(v.w) : "r"((uint32_t)p), "l"(a) : "memory");
  return v;
}
__device__ __forceinline__ void stg_cs_if(bool p, uint4* a, uint4 v) {
  asm volatile("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %0, 0;\n\t@q st.global.cs.v4.u32 [%1], {%2, %3, %4, %5};\n\t}"
               ::"r"((uint32_t)p), "l"(a), "r"(v.x), "r"(v.y), "r"(v.z), "r"(v.w) : "memory");
}
// Loads the 16-byte chunk at shared address a into x..w when p; else leaves them.
__device__ __forceinline__ void lds128_if(bool p, uint32_t a, uint32_t& x, uint32_t& y, uint32_t& z, uint32_t& w) {
  asm volatile("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %4, 0;\n\t@q ld.shared.v4.u32 {%0, %1, %2, %3}, [%5];\n\t}"
               : "+r"(x), "+r"(y), "+r"(z), "+r"(w) : "r"((uint32_t)p), "r"(a) : "memory");
}
// Atomic add of 4 to the shared word at a when p, returning the old value.
// GAS_ATOM_NOPRED (default): the atomic always executes and adds 4 or 0 — ptxas
// turns a predicated ATOMS into BSSY / BRA / ATOMS / BSYNC (3 extra
// instructions per key whose predicate is not a constant); callers guarantee
// that `a` is a valid counter address for every slot (slots past the end hold
// a copy of a real key) and ignore the result when !p. atoms_add4_pred keeps
// the predicated form (addresses that may be garbage when !p, and the kernels
// where the unpredicated form measured slower: the key-linear kernel 4.50 ->
// 4.57 ms, the split kernel's plain path on dup16 4.91 -> 4.95 ms; the value
// kernel gained 4.096 -> 4.038 ms and the batch-CDF kernel 4.51 -> 4.44 ms,
// profiles/r02_ab_atom_nopred.txt).
__device__ __forceinline__ uint32_t atoms_add4_pred(bool p, uint32_t a) {
  uint32_t v = 0;
  asm volatile("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %1, 0;\n\t@q atom.shared.add.u32 %0, [%2], 4;\n\t}"
               : "+r"(v) : "r"((uint32_t)p), "r"(a) : "memory");
  return v;
}
__device__ __forceinline__ uint32_t atoms_add4_if(bool p, uint32_t a) {
#if GAS_ATOM_NOPRED
  uint32_t v;
  asm volatile("atom.shared.add.u32 %0, [%1], %2;" : "=r"(v) : "r"(a), "r"(p ? 4u : 0u) : "memory");
  return v;
#else
  return atoms_add4_pred(p, a);
#endif
}

// ---- Control block of the 512 < n <= 1024 pipeline (sort1024.cuh): device
// workspace of one gas_sort_arrays call, followed by an array-index list of
// up to N entries.
enum : uint32_t { kS1Bucket = 0, kS1Count = 1, kS1Split = 2, kS1KeyLin = 3, kS1Cdf = 4 };
enum : uint32_t { kSplitDup = 0, kSplitSpecial = 1 };
constexpr int kCdfEntries = 512;  // batch CDF table: one entry per (sign, exponent) of the key, i.e. key >> 23
struct S1Ctl {
  uint32_t flag;      // the path that takes the whole batch (kS1*), written by the sampler
  uint32_t nlist;     // arrays the counting-sort kernel hands to the split kernel (zeroed by the sampler)
  uint32_t split_kind;  // kSplitDup / kSplitSpecial: why the sampler chose the split kernel
  uint32_t pad;
  uint2 cdf[kCdfEntries];  // (A, B) of the batch CDF map (cdf_bucket), written by the sampler
};
// The list of nlist array indices follows the control block.
__device__ __forceinline__ uint32_t* s1_list(S1Ctl* c) { return reinterpret_cast<uint32_t*>(c + 1); }
__device__ __forceinline__ const uint32_t* s1_list(const S1Ctl* c) { return reinterpret_cast<const uint32_t*>(c + 1); }
__device__ __forceinline__ void s1_push(uint32_t& count, uint32_t* list, int64_t a, int lane) {
  if (lane == 0) list[atomicAdd(&count, 1u)] = (uint32_t)a;
}

// Batch-CDF bucket map (MAP = kMapCdf): the sampler estimates, from the keys
// of its 32 sampled arrays (S keys), the distribution function of the batch at
// the 512 binade boundaries of the key space (e = key >> 23: sign and
// exponent) and writes, per entry e with c_e sampled keys and P_e sampled keys
// below it,
//     A_e = min(2^32 - 1, floor(P_e 2^32 / S)),   B_e = floor(c_e 2^16 / S).
// A key's bucket is b = (A_e + m' B_e) >> 26 with m' = the top 16 mantissa
// bits: the estimated distribution function at the key, linear inside a
// binade, times 64. For every key, 0 <= b <= 63 and b is non-decreasing in the
// key, whatever the table holds as long as it was built this way:
// A_e + (2^16 - 1) B_e < (P_e + c_e) 2^32 / S and, being an integer, is at most
// A_{e+1}. Arrays drawn from the batch's distribution (spectra intensities:
// log-normal-like, BASELINE.json spectra_intensity) then get ~n/64 keys per
// bucket, as flat data does under the value map. This is the paper's
// "sampling according to the distribution" (§9; splitters from a
// sample, Alg. 1) moved from one array to the batch.
__device__ __forceinline__ uint32_t cdf_bucket_addr(uint32_t kk, uint32_t tbl_sa, uint32_t cnt_sa) {
  uint32_t a, b;
  asm volatile("ld.shared.v2.u32 {%0, %1}, [%2];" : "=r"(a), "=r"(b) : "r"(tbl_sa + (kk >> 23) * 8u) : "memory");
  const uint32_t u = a + ((kk >> 7) & 0xFFFFu) * b;
  return cnt_sa + (u >> 26) * 4u;
}
enum : int { kMapValue = 0, kMapKeyLin = 1, kMapCdf = 2 };

// Key-linear bucket map (KL kernels): b(key) = umulhi(key - kmin, M) with
//     M = min(2^32 - 1, floor(2^38 / (kmax - kmin + 1)))   (computed rounding down),
// so 0 <= b <= 63 (x M < 2^38 for x <= kmax - kmin) and b is non-decreasing in
// the key. Keys are the totalOrder keys (ordered_key.cuh), or the raw bits of
// an all-positive finite array, so NaN, infinities and ±0 need no special
// case: the order of the keys is the order of the output (C-1).
// Key-linear buckets are uniform over the bit patterns (BASELINE.json
// uniform_bits), where value-linear buckets put nearly every key into bucket 0.
__device__ __forceinline__ uint32_t kl_mult(uint32_t kmin, uint32_t kmax) {
  const float den = __fadd_ru(__uint2float_ru(kmax - kmin), 1.0f);  // >= range + 1
  const float q = __fdiv_rz(274877906944.0f, den);                   // <= 2^38 / (range + 1)
  return q >= 4294967040.0f ? 0xFFFFFFFFu : __float2uint_rz(q);
}

#ifndef GAS_S1_PRED  // sample keys in one value bucket that send an array to the counting sort
#define GAS_S1_PRED 5
#endif
// The 32-key sample of the predictors: one key per lane, spread over the
// first 512 elements (which always exist, n > 512) so that pre-sorted arrays
// do not look skewed: VEC layout, word 0 of chunk lane + 32 (lane & 3)
// (element 4 lane + 128 (lane & 3)); scalar layout, element lane + 32 (lane & 15).
template <bool VEC>
__device__ __forceinline__ uint32_t bk_sample_key(const uint32_t (&k)[32], int lane) {
  if constexpr (VEC) {
    const uint32_t a = (lane & 1) ? k[4] : k[0], b = (lane & 1) ? k[12] : k[8];
    return (lane & 2) ? b : a;
  } else {
    const uint32_t a0 = (lane & 1) ? k[1] : k[0], a1 = (lane & 1) ? k[3] : k[2];
    const uint32_t a2 = (lane & 1) ? k[5] : k[4], a3 = (lane & 1) ? k[7] : k[6];
    const uint32_t a4 = (lane & 1) ? k[9] : k[8], a5 = (lane & 1) ? k[11] : k[10];
    const uint32_t a6 = (lane & 1) ? k[13] : k[12], a7 = (lane & 1) ? k[15] : k[14];
    const uint32_t b0 = (lane & 2) ? a1 : a0, b1 = (lane & 2) ? a3 : a2;
    const uint32_t b2 = (lane & 2) ? a5 : a4, b3 = (lane & 2) ? a7 : a6;
    const uint32_t c0 = (lane & 4) ? b1 : b0, c1 = (lane & 4) ? b3 : b2;
    return (lane & 8) ? c1 : c0;
  }
}

// Overflow predictor of the value buckets (the pipeline's sampler and the
// fused small-batch kernel): the 32-key sample k0 (one key per lane) must not
// put >= 12 keys into the 8 lowest or the 8 highest buckets (peaked values
// such as log-normal intensities), >= GAS_S1_PRED keys into one bucket, or
// repeat one value >= 3 times (duplicate-heavy arrays: a repeated value fills
// a bucket no map can split).
__device__ __forceinline__ bool bk_sample_ok(uint32_t k0, bool raw, float vmin, float s) {
  const uint32_t sb = bucket_bits(k0, vmin, s) - 0x4B000000u;
  const bool skew = __popc(__ballot_sync(0xffffffffu, sb < 8u)) >= 12 ||
                    __popc(__ballot_sync(0xffffffffu, sb > (uint32_t)GAS_BK_TOP - 8u)) >= 12;
  const int bmax = __reduce_max_sync(0xffffffffu, __popc(__match_any_sync(0xffffffffu, sb)));
  const int vmax = __reduce_max_sync(0xffffffffu, __popc(__match_any_sync(0xffffffffu, k0)));
  return !skew && bmax < GAS_S1_PRED && vmax < 3;
}

// Fixed-length arrays, 512 < n <= 1024, 16-byte-aligned rows (n % 4 == 0).
// One warp per array (persistent grid-stride). Per array:
//  1. load (8 x LDG.128 per lane); min / max of the raw bits (VIMNMX3 + REDUX).
//     All values positive and finite (the paper's data): the raw
//     bits sort as unsigned integers and are the keys ("raw" arrays); else the
//     keys are the totalOrder transform (ordered_key.cuh) and an infinity or
//     NaN sends the array to the fallback network.
//  2. bucket counter b starts at the shared address of slot 0 of bucket row b
//     and each key adds 4 to it: the atomic's old value IS the key's slot
//     address (bucket row b, rank = arrival order), and the key is stored
//     there at once. A bucket of more than 32 keys sends the array to the
//     fallback; its overflowing stores stay inside this warp's slot buffer
//     (addresses are clamped to its last word).
//  3. pad keys after the last key of each row, up to the next 16-byte chunk.
//  4. rounds: lane l sorts bucket l + 32 first, then bucket l. Only the
//     ceil(size/4) chunks holding keys are gathered: the other registers hold
//     pads (first round) or the sorted keys of bucket l + 32 (second round),
//     which all follow every key of bucket l (the map is monotone), so the
//     first size_b network outputs are bucket b sorted in both rounds.
//     Outputs are staged at slot words kBkStageWord + base_b + i.
//  5. coalesced in-place store (key -> bits for non-raw arrays).
// KL: the key-linear map (kl_mult) instead of the value map: any bit pattern
// (NaN, infinities, ±0) takes the bucket path; only an overflowing bucket sends
// the array to the fallback. Non-raw arrays stage bits, so every array leaves
// through the TMA bulk store. (The pipeline's kS1KeyLin kernel.)
// MAP = kMapCdf: the batch-CDF map (cdf_bucket_addr); the table (4 KB) is
// copied into shared memory after the per-warp areas.
template <bool PIPE, int MAP = kMapValue>
__global__ void __launch_bounds__(kBkBlock, GAS_BK_WARPS_PER_SM * 32 / kBkBlock)
    k_fixed_bucket1024(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one, const S1Ctl* ctl) {
  constexpr bool KL = MAP != kMapValue;  // keys (not values) are bucketed: every bit pattern takes the bucket path
  if (PIPE && ctl->flag != (MAP == kMapCdf ? kS1Cdf : (MAP == kMapKeyLin ? kS1KeyLin : kS1Bucket))) return;
  extern __shared__ __align__(16) uint4 bk_smem[];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const uint32_t tbl_sa = (uint32_t)__cvta_generic_to_shared(bk_smem) + (kBkBlock / 32) * kBkWarpBytes;
  if constexpr (MAP == kMapCdf) {
    for (int e = threadIdx.x; e < kCdfEntries; e += kBkBlock) {
      const uint2 v = ctl->cdf[e];
      asm volatile("st.shared.v2.u32 [%0], {%1, %2};" ::"r"(tbl_sa + e * 8u), "r"(v.x), "r"(v.y) : "memory");
    }
    __syncthreads();
  }
  const uint32_t tbl_raw = tbl_sa + 256u * 8u;  // raw (all positive) arrays: key >> 23 = (bits >> 23) + 256
  const uint32_t wsa = (uint32_t)__cvta_generic_to_shared(bk_smem) + warp * kBkWarpBytes;
  const uint32_t cnt_sa = wsa;                               // counter of bucket b at cnt_sa + b*4
  const uint32_t slot_sa = wsa + kBkCntBytes;                // slot (p, b) at slot_sa + (36 b + p)*4
  const uint32_t stage_sa = slot_sa + kBkStageWord * 4;      // output word p at stage_sa + p*4
  const uint32_t slot_last = slot_sa + kBkSlotBytes - 4;     // clamp of the scatter addresses
  uint32_t* const slot_ptr = reinterpret_cast<uint32_t*>(reinterpret_cast<unsigned char*>(bk_smem) +
                                                         warp * kBkWarpBytes + kBkCntBytes);
  const int nc = n >> 2;  // 16-byte chunks per array (> 128)
  const int64_t nwarps = (int64_t)gridDim.x * (kBkBlock / 32);
  const uint32_t cnt_b0 = cnt_sa - 0x4B000000u * 4u;  // counter address = bucket bits * 4 + cnt_b0
  const uint32_t row0 = slot_sa + lane * (kBkRowWords * 4);  // this lane's rows: buckets lane, lane + 32
  const uint32_t row1 = row0 + 32 * (kBkRowWords * 4);

  for (int64_t a = (int64_t)blockIdx.x * (kBkBlock / 32) + warp; a < N; a += nwarps) {
    uint4* const dst = reinterpret_cast<uint4*>(d + a * (int64_t)n);
    // ---- a2: stage in (raw bits); chunks q >= 4 may lie past the end (n > 512)
    uint32_t k[32];
#pragma unroll
    for (int q = 0; q < 8; ++q) {
      const int c = lane + 32 * q;
      const uint4 v = q < 4 ? ld_stream(dst + c) : ldg_cs_if(c < nc, dst + c);
      k[4 * q] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
    }
#if GAS_BK_PREFETCH
    // warm L2 with this warp's next array (one TMA bulk prefetch)
    if (GAS_BK_ELECT) {
      bulk_prefetch_elect(a + GAS_BK_PREFETCH * nwarps < N, d + (a + GAS_BK_PREFETCH * nwarps) * (int64_t)n, (uint32_t)n * 4u);
    } else if (lane == 0 && a + GAS_BK_PREFETCH * nwarps < N) {
      asm volatile("cp.async.bulk.prefetch.L2.global [%0], %1;" ::"l"(d + (a + GAS_BK_PREFETCH * nwarps) * (int64_t)n),
                   "r"((uint32_t)n * 4u) : "memory");
    }
#endif
#if GAS_BK_TMA_STORE
    // the previous bulk store has read the staging (the lane that issued it waits)
    if (GAS_BK_ELECT) bulk_wait_read_elect();
    else if (lane == 0) asm volatile("cp.async.bulk.wait_group.read 0;" ::: "memory");
    __syncwarp();
#endif
    // slots past the end repeat k[0] so that min / max need no predicates
#pragma unroll
    for (int q = 4; q < 8; ++q) {
      const bool v = lane + 32 * q < nc;
#pragma unroll
      for (int j = 0; j < 4; ++j) k[4 * q + j] = v ? k[4 * q + j] : k[0];
    }
    // ---- bucket map parameters
    uint32_t umin = k[0], umax = k[0];
#pragma unroll
    for (int r = 1; r < 31; r += 2) {
      umin = __vimin3_u32(umin, k[r], k[r + 1]);
      umax = __vimax3_u32(umax, k[r], k[r + 1]);
    }
    umin = __reduce_min_sync(0xffffffffu, min(umin, k[31]));
    umax = __reduce_max_sync(0xffffffffu, max(umax, k[31]));
    const bool raw = umin > 0u && umax < 0x7F800000u;  // every value positive and finite
    bool use_buckets = true;
    float vmin = 0.0f, s = 0.0f;
    uint32_t klo = umin, mk = 0;  // KL: key minimum and multiplier
    if (!raw) {  // min / max in key space; an infinity or NaN (either sign) -> fallback
      uint32_t kmin = 0xFFFFFFFFu, kmax = 0u;
#pragma unroll
      for (int r = 0; r < 32; ++r) {
        const uint32_t kk = key_from_bits(k[r]);
        kmin = min(kmin, kk);
        kmax = max(kmax, kk);
      }
      kmin = __reduce_min_sync(0xffffffffu, kmin);
      kmax = __reduce_max_sync(0xffffffffu, kmax);
      if constexpr (KL) {
        klo = kmin;
        umax = kmax;
      } else {
        use_buckets = kmin > 0x007FFFFFu && kmax < 0xFF800000u;
        umin = bits_from_key(kmin);
        umax = bits_from_key(kmax);
      }
    }
    if constexpr (MAP == kMapKeyLin) {
      mk = kl_mult(klo, umax);
    } else if constexpr (MAP == kMapCdf) {
      (void)mk;
    } else {
      vmin = __uint_as_float(umin);
      const float range = __fsub_rn(__uint_as_float(umax), vmin);
      s = __fdiv_rn((float)GAS_BK_TOP, range);
      use_buckets = use_buckets && range > 0.0f && range <= 3.402823466e38f && s <= 3.402823466e38f;
    }
    uint32_t t0 = 0, t1 = 0, base0 = 0, base1 = 0;
    if (use_buckets) {
      // lane l owns buckets l (row l) and l + 32 (row 32 + l)
      sts32(cnt_sa + lane * 4, row0);
      sts32(cnt_sa + 128 + lane * 4, row1);
      __syncwarp();
      // ---- rank + scatter: the atomic returns the key's slot address
      // (in groups of GAS_BK_GROUP keys: the atomics of a group are in flight together)
      if constexpr (MAP == kMapCdf) {
        if (raw) {
#pragma unroll
          for (int g = 0; g < 32; g += GAS_BK_GROUP) {
            uint32_t sa[GAS_BK_GROUP];
#pragma unroll
            for (int r = g; r < g + GAS_BK_GROUP; ++r)
              sa[r - g] = atoms_add4_if((r >> 2) < 4 || lane + 32 * (r >> 2) < nc, cdf_bucket_addr(k[r], tbl_raw, cnt_sa));
#pragma unroll
            for (int r = g; r < g + GAS_BK_GROUP; ++r)
              sts32_if((r >> 2) < 4 || lane + 32 * (r >> 2) < nc, min(sa[r - g], slot_last), k[r]);
          }
        } else {
#pragma unroll
          for (int g = 0; g < 32; g += GAS_BK_GROUP) {
            uint32_t sa[GAS_BK_GROUP], kk[GAS_BK_GROUP];
#pragma unroll
            for (int r = g; r < g + GAS_BK_GROUP; ++r) {
              kk[r - g] = key_from_bits(k[r]);
              sa[r - g] = atoms_add4_if((r >> 2) < 4 || lane + 32 * (r >> 2) < nc, cdf_bucket_addr(kk[r - g], tbl_sa, cnt_sa));
            }
#pragma unroll
            for (int r = g; r < g + GAS_BK_GROUP; ++r)
              sts32_if((r >> 2) < 4 || lane + 32 * (r >> 2) < nc, min(sa[r - g], slot_last), kk[r - g]);
          }
        }
      } else if constexpr (KL) {
        if (raw) {
#pragma unroll
          for (int g = 0; g < 32; g += GAS_BK_GROUP) {
            uint32_t sa[GAS_BK_GROUP];
#pragma unroll
            for (int r = g; r < g + GAS_BK_GROUP; ++r)
              sa[r - g] = atoms_add4_pred((r >> 2) < 4 || lane + 32 * (r >> 2) < nc, __umulhi(k[r] - klo, mk) * 4u + cnt_sa);
#pragma unroll
            for (int r = g; r < g + GAS_BK_GROUP; ++r)
              sts32_if((r >> 2) < 4 || lane + 32 * (r >> 2) < nc, min(sa[r - g], slot_last), k[r]);
          }
        } else {
#pragma unroll
          for (int g = 0; g < 32; g += GAS_BK_GROUP) {
            uint32_t sa[GAS_BK_GROUP], kk[GAS_BK_GROUP];
#pragma unroll
            for (int r = g; r < g + GAS_BK_GROUP; ++r) {
              kk[r - g] = key_from_bits(k[r]);
              sa[r - g] = atoms_add4_pred((r >> 2) < 4 || lane + 32 * (r >> 2) < nc, __umulhi(kk[r - g] - klo, mk) * 4u + cnt_sa);
            }
#pragma unroll
            for (int r = g; r < g + GAS_BK_GROUP; ++r)
              sts32_if((r >> 2) < 4 || lane + 32 * (r >> 2) < nc, min(sa[r - g], slot_last), kk[r - g]);
          }
        }
      } else if (raw) {
#pragma unroll
        for (int g = 0; g < 32; g += GAS_BK_GROUP) {
          uint32_t sa[GAS_BK_GROUP];
#pragma unroll
          for (int r = g; r < g + GAS_BK_GROUP; ++r)
            sa[r - g] = atoms_add4_if((r >> 2) < 4 || lane + 32 * (r >> 2) < nc, bucket_bits(k[r], vmin, s) * 4u + cnt_b0);
#pragma unroll
          for (int r = g; r < g + GAS_BK_GROUP; ++r)
            sts32_if((r >> 2) < 4 || lane + 32 * (r >> 2) < nc, min(sa[r - g], slot_last), k[r]);
        }
      } else {
#pragma unroll
        for (int g = 0; g < 32; g += GAS_BK_GROUP) {
          uint32_t sa[GAS_BK_GROUP];
#pragma unroll
          for (int r = g; r < g + GAS_BK_GROUP; ++r)
            sa[r - g] = atoms_add4_if((r >> 2) < 4 || lane + 32 * (r >> 2) < nc, bucket_bits(k[r], vmin, s) * 4u + cnt_b0);
#pragma unroll
          for (int r = g; r < g + GAS_BK_GROUP; ++r)
            sts32_if((r >> 2) < 4 || lane + 32 * (r >> 2) < nc, min(sa[r - g], slot_last), key_from_bits(k[r]));
        }
      }
      __syncwarp();
      t0 = (lds32(cnt_sa + lane * 4) - row0) >> 2;
      t1 = (lds32(cnt_sa + 128 + lane * 4) - row1) >> 2;
      use_buckets = __all_sync(0xffffffffu, t0 <= 32u && t1 <= 32u);
      if (use_buckets) {
        // pads after the last key of each row, up to its 16-byte chunk boundary
#pragma unroll
        for (int j = 0; j < 3; ++j) {
          sts32_if(((t0 + j) & 3u) != 0u, row0 + (t0 + j) * 4, kPadKey);
          sts32_if(((t1 + j) & 3u) != 0u, row1 + (t1 + j) * 4, kPadKey);
        }
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
        __syncwarp();
      }
    }

    if (use_buckets) {
      // ---- two bucket rounds per lane (rolled: the hot code stays in the
      // instruction cache): bucket lane + 32, then bucket lane
#pragma unroll 1
      for (int rho = 0; rho < 2; ++rho) {
        const uint32_t tb = rho ? t0 : t1;
        const uint32_t row = rho ? row0 : row1;
        const uint32_t ob = stage_sa + (rho ? base0 : base1) * 4;
        if (rho == 0) {
#pragma unroll
          for (int i = 0; i < 32; ++i) k[i] = kPadKey;
        }
#pragma unroll
        for (int q = 0; q < 8; ++q) lds128_if(4u * q < tb, row + q * 16, k[4 * q], k[4 * q + 1], k[4 * q + 2], k[4 * q + 3]);
        __syncwarp();  // rows 32..63 are drained before any output is staged over them
        sortn_bk<32>(k, one);
        if (GAS_BK_MASKSTORE && MAP != kMapValue) {  // (the value kernel measured 0.5% slower with it)
          uint32_t* const sw = reinterpret_cast<uint32_t*>(bk_smem);
          const uint32_t w0 = (ob - (uint32_t)__cvta_generic_to_shared(bk_smem)) >> 2;
          if (MAP == kMapKeyLin && GAS_BK_TMA_STORE && !raw) stage_first<true>(sw, w0, tb, k);  // bits (k keeps the keys)
          else stage_first<false>(sw, w0, tb, k);
        } else if (MAP == kMapKeyLin && GAS_BK_TMA_STORE && !raw) {  // stage bits (k keeps the keys: they pad the second round)
#pragma unroll
          for (int i = 0; i < 32; ++i) sts32_if((uint32_t)i < tb, ob + i * 4, bits_from_key(k[i]));
        } else {
#pragma unroll
          for (int i = 0; i < 32; ++i) sts32_if((uint32_t)i < tb, ob + i * 4, k[i]);
        }
      }
#if GAS_BK_TMA_STORE
      if (raw || MAP == kMapKeyLin) {  // the staged array is contiguous: one TMA bulk store (the copy engine reads shared memory)
        asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
        __syncwarp();
        if (GAS_BK_ELECT) {
          bulk_store_elect(dst, stage_sa, (uint32_t)n * 4u);
        } else if (lane == 0) {
          asm volatile("cp.async.bulk.global.shared::cta.bulk_group [%0], [%1], %2;"
                       ::"l"(dst), "r"(stage_sa), "r"((uint32_t)n * 4u) : "memory");
          asm volatile("cp.async.bulk.commit_group;" ::: "memory");
        }
      } else {
#else
      __syncwarp();
      if (raw) {
#pragma unroll
        for (int q = 0; q < 8; ++q) {
          const int c = lane + 32 * q;
          stg_cs_if(q < 4 || c < nc, dst + c, lds128(stage_sa + c * 16));
        }
      } else {
#endif
        __syncwarp();
#pragma unroll
        for (int q = 0; q < 8; ++q) {
          const int c = lane + 32 * q;
          uint4 v = lds128(stage_sa + c * 16);
          v.x = bits_from_key(v.x); v.y = bits_from_key(v.y); v.z = bits_from_key(v.z); v.w = bits_from_key(v.w);
          stg_cs_if(q < 4 || c < nc, dst + c, v);
        }
      }
    } else {
      __syncwarp();  // the fallback's scratch overlaps the slot buffer
      bucket1024_fallback(k, dst, nc, lane, slot_ptr, one);
    }
    __syncwarp();
  }
#if GAS_BK_TMA_STORE
  if (lane == 0) asm volatile("cp.async.bulk.wait_group 0;" ::: "memory");  // stores complete before the CTA exits
#endif
}

// The same kernel for rows at any 4-byte alignment (n % 4 != 0 or an
// unaligned base; instantiated with VEC = false): key r of a lane is element
// lane + 32 r (4-byte accesses). Kept apart from k_fixed_bucket1024 so that the
// 16-byte kernel's register allocation stays as measured (a merged template
// spilled 12 bytes per array: 4.21 -> 4.31 ms).
template <bool VEC, bool PIPE>
__global__ void __launch_bounds__(kBkBlock, GAS_BK_WARPS_PER_SM * 32 / kBkBlock)
    k_fixed_bucket1024_any(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one, const S1Ctl* ctl) {
  if (PIPE && ctl->flag != kS1Bucket) return;  // pipeline (sort1024.cuh): another kernel takes this batch
  extern __shared__ __align__(16) uint4 bk_smem[];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const uint32_t wsa = (uint32_t)__cvta_generic_to_shared(bk_smem) + warp * kBkWarpBytes;
  const uint32_t cnt_sa = wsa;                               // counter of bucket b at cnt_sa + b*4
  const uint32_t slot_sa = wsa + kBkCntBytes;                // slot (p, b) at slot_sa + (36 b + p)*4
  const uint32_t stage_sa = slot_sa + kBkStageWord * 4;      // output word p at stage_sa + p*4
  const uint32_t slot_last = slot_sa + kBkSlotBytes - 4;     // clamp of the scatter addresses
  uint32_t* const slot_ptr = reinterpret_cast<uint32_t*>(reinterpret_cast<unsigned char*>(bk_smem) +
                                                         warp * kBkWarpBytes + kBkCntBytes);
  const int nc = n >> 2;  // 16-byte chunks per array (> 128)
  const int64_t nwarps = (int64_t)gridDim.x * (kBkBlock / 32);
  const uint32_t cnt_b0 = cnt_sa - 0x4B000000u * 4u;  // counter address = bucket bits * 4 + cnt_b0
  const uint32_t row0 = slot_sa + lane * (kBkRowWords * 4);  // this lane's rows: buckets lane, lane + 32
  const uint32_t row1 = row0 + 32 * (kBkRowWords * 4);

  // key r of this lane lies inside the array (always for r < 16: n > 512)
  auto valid = [&](int r) -> bool {
    return VEC ? ((r >> 2) < 4 || lane + 32 * (r >> 2) < nc) : (r < 16 || lane + 32 * r < n);
  };
  for (int64_t a = (int64_t)blockIdx.x * (kBkBlock / 32) + warp; a < N; a += nwarps) {
    uint32_t* const arr = d + a * (int64_t)n;
    uint4* const dst = reinterpret_cast<uint4*>(arr);
    // ---- a2: stage in (raw bits); keys r >= 16 may lie past the end (n > 512)
    uint32_t k[32];
    if constexpr (VEC) {
#pragma unroll
      for (int q = 0; q < 8; ++q) {
        const int c = lane + 32 * q;
        const uint4 v = q < 4 ? ld_stream(dst + c) : ldg_cs_if(c < nc, dst + c);
        k[4 * q] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
      }
    } else {
#pragma unroll
      for (int r = 0; r < 32; ++r) k[r] = valid(r) ? ld_stream(arr + lane + 32 * r) : 0u;
    }
#if GAS_BK_PREFETCH
    if (lane == 0 && a + GAS_BK_PREFETCH * nwarps < N) {  // warm L2 with this warp's next array (one TMA bulk prefetch)
      if constexpr (VEC)
        asm volatile("cp.async.bulk.prefetch.L2.global [%0], %1;" ::"l"(d + (a + GAS_BK_PREFETCH * nwarps) * (int64_t)n),
                     "r"((uint32_t)n * 4u) : "memory");
      else
        prefetch_l2(d + (a + GAS_BK_PREFETCH * nwarps) * (int64_t)n, n);
    }
#endif
    // slots past the end repeat k[0] so that min / max need no predicates
#pragma unroll
    for (int r = 16; r < 32; ++r) k[r] = valid(r) ? k[r] : k[0];
    // ---- bucket map parameters
    uint32_t umin = k[0], umax = k[0];
#pragma unroll
    for (int r = 1; r < 31; r += 2) {
      umin = __vimin3_u32(umin, k[r], k[r + 1]);
      umax = __vimax3_u32(umax, k[r], k[r + 1]);
    }
    umin = __reduce_min_sync(0xffffffffu, min(umin, k[31]));
    umax = __reduce_max_sync(0xffffffffu, max(umax, k[31]));
    const bool raw = umin > 0u && umax < 0x7F800000u;  // every value positive and finite
    bool use_buckets = true;
    if (!raw) {  // min / max in key space; an infinity or NaN (either sign) -> fallback
      uint32_t kmin = 0xFFFFFFFFu, kmax = 0u;
#pragma unroll
      for (int r = 0; r < 32; ++r) {
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
    const float s = __fdiv_rn((float)GAS_BK_TOP, range);
    use_buckets = use_buckets && range > 0.0f && range <= 3.402823466e38f && s <= 3.402823466e38f;
    uint32_t t0 = 0, t1 = 0, base0 = 0, base1 = 0;
    if (use_buckets) {
      // lane l owns buckets l (row l) and l + 32 (row 32 + l)
      sts32(cnt_sa + lane * 4, row0);
      sts32(cnt_sa + 128 + lane * 4, row1);
      __syncwarp();
      // ---- rank + scatter: the atomic returns the key's slot address
      // (in groups of GAS_BK_GROUP keys: the atomics of a group are in flight together)
      if (raw) {
#pragma unroll
        for (int g = 0; g < 32; g += GAS_BK_GROUP) {
          uint32_t sa[GAS_BK_GROUP];
#pragma unroll
          for (int r = g; r < g + GAS_BK_GROUP; ++r)
            sa[r - g] = atoms_add4_if(valid(r), bucket_bits(k[r], vmin, s) * 4u + cnt_b0);
#pragma unroll
          for (int r = g; r < g + GAS_BK_GROUP; ++r)
            sts32_if(valid(r), min(sa[r - g], slot_last), k[r]);
        }
      } else {
#pragma unroll
        for (int g = 0; g < 32; g += GAS_BK_GROUP) {
          uint32_t sa[GAS_BK_GROUP];
#pragma unroll
          for (int r = g; r < g + GAS_BK_GROUP; ++r)
            sa[r - g] = atoms_add4_if(valid(r), bucket_bits(k[r], vmin, s) * 4u + cnt_b0);
#pragma unroll
          for (int r = g; r < g + GAS_BK_GROUP; ++r)
            sts32_if(valid(r), min(sa[r - g], slot_last), key_from_bits(k[r]));
        }
      }
      __syncwarp();
      t0 = (lds32(cnt_sa + lane * 4) - row0) >> 2;
      t1 = (lds32(cnt_sa + 128 + lane * 4) - row1) >> 2;
      use_buckets = __all_sync(0xffffffffu, t0 <= 32u && t1 <= 32u);
      if (use_buckets) {
        // pads after the last key of each row, up to its 16-byte chunk boundary
#pragma unroll
        for (int j = 0; j < 3; ++j) {
          sts32_if(((t0 + j) & 3u) != 0u, row0 + (t0 + j) * 4, kPadKey);
          sts32_if(((t1 + j) & 3u) != 0u, row1 + (t1 + j) * 4, kPadKey);
        }
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
        __syncwarp();
      }
    }

    if (use_buckets) {
      // ---- two bucket rounds per lane (rolled: the hot code stays in the
      // instruction cache): bucket lane + 32, then bucket lane
#pragma unroll 1
      for (int rho = 0; rho < 2; ++rho) {
        const uint32_t tb = rho ? t0 : t1;
        const uint32_t row = rho ? row0 : row1;
        const uint32_t ob = stage_sa + (rho ? base0 : base1) * 4;
        if (rho == 0) {
#pragma unroll
          for (int i = 0; i < 32; ++i) k[i] = kPadKey;
        }
#pragma unroll
        for (int q = 0; q < 8; ++q) lds128_if(4u * q < tb, row + q * 16, k[4 * q], k[4 * q + 1], k[4 * q + 2], k[4 * q + 3]);
        __syncwarp();  // rows 32..63 are drained before any output is staged over them
        sortn_bk<32>(k, one);
#pragma unroll
        for (int i = 0; i < 32; ++i) sts32_if((uint32_t)i < tb, ob + i * 4, k[i]);
      }
      __syncwarp();
      if constexpr (!VEC) {
        if (raw) {
#pragma unroll
          for (int r = 0; r < 32; ++r)
            if (valid(r)) st_stream(arr + lane + 32 * r, lds32(stage_sa + (lane + 32 * r) * 4));
        } else {
#pragma unroll
          for (int r = 0; r < 32; ++r)
            if (valid(r)) st_stream(arr + lane + 32 * r, bits_from_key(lds32(stage_sa + (lane + 32 * r) * 4)));
        }
      } else if (raw) {
#pragma unroll
        for (int q = 0; q < 8; ++q) {
          const int c = lane + 32 * q;
          stg_cs_if(q < 4 || c < nc, dst + c, lds128(stage_sa + c * 16));
        }
      } else {
#pragma unroll
        for (int q = 0; q < 8; ++q) {
          const int c = lane + 32 * q;
          uint4 v = lds128(stage_sa + c * 16);
          v.x = bits_from_key(v.x); v.y = bits_from_key(v.y); v.z = bits_from_key(v.z); v.w = bits_from_key(v.w);
          stg_cs_if(q < 4 || c < nc, dst + c, v);
        }
      }
    } else {
      __syncwarp();  // the fallback's scratch overlaps the slot buffer
      if constexpr (VEC) bucket1024_fallback(k, dst, nc, lane, slot_ptr, one);
      else bucket1024_fallback_scalar(k, arr, n, lane, slot_ptr, one);
    }
    __syncwarp();
  }
}

}  // namespace gas
