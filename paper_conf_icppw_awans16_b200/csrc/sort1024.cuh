// sort1024.cuh — the default sort of one array of 512 < n <= 1024 keys by one
// warp (the n = 1000 headline of BASELINE.json configs[1]): the value-bucket
// kernel of bucket1024.cuh where its buckets fit, the counting sort of
// cw1024.cuh where they do not, the 1024-key network only as a last resort.
//
// Per array (warp-uniform decisions, the array stays in registers throughout):
//  1. load; min / max of the raw bits (and of the ordered keys when some value
//     is negative, zero, infinite or NaN).
//  2. finite values: 64 value-linear buckets (bucket1024.cuh) unless a 32-key
//     sample (bk_sample_key, bucket1024.cuh) already puts >= GAS_S1_PRED
//     samples in one bucket (peaked values such as log-normal spectra
//     intensities, duplicate-heavy arrays: a 32-slot bucket would overflow).
//     Measured on the paper's uniform data: 0.5% of arrays overflow anyway.
//  3. anything else, and every bucket overflow: the counting sort on 2048
//     key-linear fine bins (cw1024.cuh), whose cost does not depend on the
//     value distribution; arrays whose sample holds >= 2 NaN / infinity / -0
//     patterns go straight to the network (such arrays usually hold many ±inf
//     and ±0, single keys that share fine bins with NaNs and subnormals, a
//     case the counting sort's repair step cannot fix).
//  4. the counting sort's own check failing: the 1024-key network
//     (warp1024.cuh) from the same registers.
// Every branch ends in the same in-place store; the output is the unique
// totalOrder arrangement (C-1) whichever branch ran.
// `mode` (tests and ablations, GAS_SORT1024_MODE): 0 = the decisions above;
// 1 = every array through the counting sort; 2 = every array through the
// network; 3 = buckets without the predictor.
#pragma once
#include <cstdint>

#include "cw1024.cuh"

namespace gas {

#ifndef GAS_S1_BLOCK
#define GAS_S1_BLOCK 640  // 20 warps per SM at <= 96 registers (the counting sort's best: 768 / 80 spills)
#endif
#ifndef GAS_S1_NO_CW
#define GAS_S1_NO_CW 0
#endif
constexpr int kS1Block = GAS_S1_BLOCK;
constexpr int kS1SmemBytes = (kS1Block / 32) * kBkWarpBytes;
static_assert(kBkWarpBytes >= kCwWarpBytes, "the counting sort reuses the bucket kernel's per-warp area");

// VEC: 16-byte-aligned rows (n % 4 == 0), key r of a lane is word r % 4 of
// chunk lane + 32 (r / 4); else any 4-byte alignment, key r is element lane + 32 r.
template <bool VEC>
__global__ void __launch_bounds__(kS1Block, 1)
    k_fixed_sort1024(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one, int mode) {
  extern __shared__ __align__(16) uint4 s1_smem[];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const uint32_t wsa = (uint32_t)__cvta_generic_to_shared(s1_smem) + warp * kBkWarpBytes;
  const uint32_t cnt_sa = wsa;                               // counter of bucket b at cnt_sa + b*4
  const uint32_t slot_sa = wsa + kBkCntBytes;                // slot (p, b) at slot_sa + (36 b + p)*4
  const uint32_t stage_sa = slot_sa + kBkStageWord * 4;      // output word p at stage_sa + p*4
  const uint32_t slot_last = slot_sa + kBkSlotBytes - 4;     // clamp of the scatter addresses
  unsigned char* const wptr = reinterpret_cast<unsigned char*>(s1_smem) + warp * kBkWarpBytes;
  uint32_t* const slot_ptr = reinterpret_cast<uint32_t*>(wptr + kBkCntBytes);
  const int nc = n >> 2;  // 16-byte chunks per array (VEC)
  const int64_t nwarps = (int64_t)gridDim.x * (kS1Block / 32);
  const uint32_t cnt_b0 = cnt_sa - 0x4B000000u * 4u;  // counter address = bucket bits * 4 + cnt_b0
  const uint32_t row0 = slot_sa + lane * (kBkRowWords * 4);  // this lane's rows: buckets lane, lane + 32
  const uint32_t row1 = row0 + 32 * (kBkRowWords * 4);

  auto valid = [&](int r) -> bool { return cw_valid<VEC>(r, lane, n); };
  for (int64_t a = (int64_t)blockIdx.x * (kS1Block / 32) + warp; a < N; a += nwarps) {
    uint32_t* const arr = d + a * (int64_t)n;
    uint4* const dst = reinterpret_cast<uint4*>(arr);
    // ---- 1. stage in (raw bits); keys past the end are copies of k[0]
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
    if (lane == 0 && a + nwarps < N) {  // warm L2 with this warp's next array (one TMA bulk prefetch)
      if constexpr (VEC)
        asm volatile("cp.async.bulk.prefetch.L2.global [%0], %1;" ::"l"(d + (a + nwarps) * (int64_t)n),
                     "r"((uint32_t)n * 4u) : "memory");
      else
        prefetch_l2(d + (a + nwarps) * (int64_t)n, n);
    }
#endif
#pragma unroll
    for (int r = 16; r < 32; ++r) k[r] = valid(r) ? k[r] : k[0];
    uint32_t umin = k[0], umax = k[0];
#pragma unroll
    for (int r = 1; r < 31; r += 2) {
      umin = __vimin3_u32(umin, k[r], k[r + 1]);
      umax = __vimax3_u32(umax, k[r], k[r + 1]);
    }
    umin = __reduce_min_sync(0xffffffffu, min(umin, k[31]));
    umax = __reduce_max_sync(0xffffffffu, max(umax, k[31]));
    const bool raw = umin > 0u && umax < 0x7F800000u;  // every value positive and finite
    bool finite = true;
    uint32_t vlo = umin, vhi = umax;  // value range of the bucket map (as float bits)
    if (!raw) {  // min / max in key space
      uint32_t kmin = 0xFFFFFFFFu, kmax = 0u;
#pragma unroll
      for (int r = 0; r < 32; ++r) {
        const uint32_t kk = key_from_bits(k[r]);
        kmin = min(kmin, kk);
        kmax = max(kmax, kk);
      }
      kmin = __reduce_min_sync(0xffffffffu, kmin);
      kmax = __reduce_max_sync(0xffffffffu, kmax);
      finite = kmin > 0x007FFFFFu && kmax < 0xFF800000u;
      vlo = bits_from_key(kmin);
      vhi = bits_from_key(kmax);
    }
    const float vmin = __uint_as_float(vlo);
    const float range = __fsub_rn(__uint_as_float(vhi), vmin);
    const float s = __fdiv_rn((float)GAS_BK_TOP, range);
    bool use_buckets = mode != 1 && mode != 2 && finite && range > 0.0f && range <= 3.402823466e38f &&
                       s <= 3.402823466e38f;
    // ---- 2. predictor: the sample's most populated bucket
    if (use_buckets && mode != 3) use_buckets = bk_sample_ok(bk_sample_key<VEC>(k, lane), raw, vmin, s);
    uint32_t t0 = 0, t1 = 0, base0 = 0, base1 = 0;
    if (use_buckets) {
      // lane l owns buckets l (row l) and l + 32 (row 32 + l)
      sts32(cnt_sa + lane * 4, row0);
      sts32(cnt_sa + 128 + lane * 4, row1);
      __syncwarp();
      // rank + scatter: the atomic returns the key's slot address
      if (raw) {
#pragma unroll
        for (int g = 0; g < 32; g += GAS_BK_GROUP) {
          uint32_t sa[GAS_BK_GROUP];
#pragma unroll
          for (int r = g; r < g + GAS_BK_GROUP; ++r)
            sa[r - g] = atoms_add4_if(valid(r), bucket_bits(k[r], vmin, s) * 4u + cnt_b0);
#pragma unroll
          for (int r = g; r < g + GAS_BK_GROUP; ++r) sts32_if(valid(r), min(sa[r - g], slot_last), k[r]);
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
      // two bucket rounds per lane (rolled: the hot code stays in the
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
        if (GAS_BK_MASKSTORE) {
          stage_first<false>(reinterpret_cast<uint32_t*>(s1_smem), (ob - (uint32_t)__cvta_generic_to_shared(s1_smem)) >> 2, tb, k);
        } else {
#pragma unroll
          for (int i = 0; i < 32; ++i) sts32_if((uint32_t)i < tb, ob + i * 4, k[i]);
        }
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
      __syncwarp();  // the other branches reuse this warp's shared area
      // ---- 3. / 4. counting sort, or the network for special-heavy samples:
      // sample keys that are an infinity, a NaN or -0 (the two paths must not
      // mix on one SM: together they overflow the instruction cache)
      const uint32_t sk = bk_sample_key<VEC>(k, lane);
      const bool special = ((sk >> 23) & 0xFFu) == 0xFFu || sk == 0x80000000u;
      if (mode == 2 || (mode != 1 && !raw && __popc(__ballot_sync(0xffffffffu, special)) >= 2) || GAS_S1_NO_CW) {
        if constexpr (VEC) bucket1024_fallback(k, dst, nc, lane, slot_ptr, one);
        else bucket1024_fallback_scalar(k, arr, n, lane, slot_ptr, one);
      } else {
        cw_sort_warp<VEC>(k, raw, umin, umax, 0u, arr, n, lane, wsa, wsa + kCwCntBytes,
                          reinterpret_cast<uint32_t*>(wptr + kCwCntBytes), one);
      }
    }
    __syncwarp();
  }
}


// ---------------------------------------------------------------------------
// The pipeline used for large batches (host: k_1024.cu). One kernel that holds
// the bucket path, the counting sort and the network runs slower than each
// path alone: on one SM the hot code of two paths overflows the 32 KB
// instruction cache (ncu: "no instruction" stalls up to 86% of warp stall
// samples when arrays of one batch alternate between the counting sort and
// the network). So each path is its own kernel, and the batch's work is
// routed on the device, with no host synchronisation:
//   1. k_s1_sample: 32 warps load 32 arrays spread over the batch and vote
//      for the path each would take (the same tests as the kernels below);
//      the majority goes to ctl->flag.
//   2. k_fixed_bucket1024<PIPE = true> (bucket1024.cuh): runs the batch when
//      flag == bucket, unchanged from the stand-alone kernel (its few
//      overflowing / NaN arrays take its inline network).
//   3. k_s1_count: the counting sort over the whole batch when flag == count;
//      special-heavy arrays go to a list; arrays failing its own check are
//      finished by the network inline (rare).
//   2b. k_fixed_bucket1024<PIPE, KL = true>: the same kernel with the
//      key-linear map (flag == keylin: the sample does not fit value buckets
//      but fits key-linear ones, e.g. arrays of arbitrary bit patterns).
//   4. k_s1_split (split1024.cuh): value buckets with special-value runs and
//      equal-key runs, over the whole batch (flag == split: NaN / inf / ±0
//      mixes, duplicate-heavy data) or over that list (its arrays are read
//      from HBM a second time); its own leftovers take the network inline.
// Kernels not chosen exit at once (a few microseconds each).

// The class an array votes for: special-heavy sample -> split; finite values
// whose 32-key sample fits the buckets -> bucket; duplicate-heavy samples
// whose repeated values each fill a bucket of their own -> split; else the
// counting sort.
__device__ __forceinline__ uint32_t s1_sample_special(uint32_t k0) {
  const bool special = ((k0 >> 23) & 0xFFu) == 0xFFu || k0 == 0x80000000u;  // inf / NaN / -0
  return __popc(__ballot_sync(0xffffffffu, special));
}

// Duplicate-heavy sample the split kernel's equal-key runs can take: some
// value appears >= 3 times among the 32 sample keys, and every sample bucket
// holds a single value (a bucket overflowing with two values would not fold).
__device__ __forceinline__ bool bk_sample_dup(uint32_t k0, float vmin, float s) {
  const uint32_t sb = bucket_bits(k0, vmin, s) - 0x4B000000u;
  const uint32_t mv = __match_any_sync(0xffffffffu, k0);
  const bool single = __all_sync(0xffffffffu, __match_any_sync(0xffffffffu, sb) == mv);
  return single && __reduce_max_sync(0xffffffffu, __popc(mv)) >= 3;
}

// One block of 32 warps; warp w samples array floor(w N / 32).
//  1. every sampled key goes into a 512-bin histogram of key >> 23 (sign and
//     exponent of the totalOrder key); threads 0..511 scan it and write the
//     batch-CDF table of cdf_bucket_addr (bucket1024.cuh) to ctl->cdf;
//  2. each warp counts, in shared memory, the exact bucket sizes its array
//     gets under the value map (bk kernel), the key-linear map (KL kernel)
//     and the batch-CDF map (CDF kernel).
// The batch goes to
//   the value buckets     when >= 26 of 32 sampled arrays fit them (<= 32 keys
//                         per bucket; an overflowing array costs the bucket
//                         attempt plus the 1024-key network, ~1.8x),
//   the key-linear ones   when >= 27 fit those,
//   the batch-CDF ones    when >= 27 fit those,
//   else the split kernel or the counting sort, by the majority of the
//   sampled arrays' votes (special-heavy or duplicate-heavy -> split).
// `force` (<= kS1Cdf; tests and ablations, GAS_S1_FORCE) overrides the
// choice. The block also zeroes the list counter (no other initialisation of
// the workspace is needed).
template <bool VEC>
__global__ void __launch_bounds__(1024, 1) k_s1_sample(const uint32_t* __restrict__ d, int64_t N, int n, S1Ctl* ctl,
                                                           uint32_t force) {
  __shared__ uint32_t votes[6];  // [0] value fit, [1] key-linear fit, [2] count, [3] split, [4] batch-CDF fit, [5] special-heavy
  __shared__ uint32_t hist[32][192];  // per warp: value-bucket, key-linear and batch-CDF bucket sizes
  __shared__ uint32_t h512[kCdfEntries];
  __shared__ __align__(8) uint2 tbl[kCdfEntries];
  __shared__ uint32_t part[kCdfEntries / 32];
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  if (threadIdx.x < 6) votes[threadIdx.x] = 0;
  if (threadIdx.x < kCdfEntries) h512[threadIdx.x] = 0;
  __syncthreads();
  const int64_t S = N < 32 ? N : 32;  // arrays sampled
  const bool active = (int64_t)w < S;
  const int64_t a = (N <= 32) ? w : (int64_t)(((__int128)w * N) >> 5);
  const uint32_t* arr = d + (active ? a : 0) * (int64_t)n;
  uint32_t k[32];
  uint32_t* const h = hist[w];
  // ---- 1. each sampled array: exact bucket sizes under the value and key-linear maps
  if (active) {
#pragma unroll
    for (int r = 0; r < 32; ++r) {
      const bool v = cw_valid<VEC>(r, lane, n);
      const int e = VEC ? 4 * (lane + 32 * (r >> 2)) + (r & 3) : lane + 32 * r;
      k[r] = v ? __ldcs(arr + e) : 0u;
    }
#pragma unroll
    for (int r = 16; r < 32; ++r) k[r] = cw_valid<VEC>(r, lane, n) ? k[r] : k[0];
    uint32_t umin = k[0], umax = k[0], kmin = 0xFFFFFFFFu, kmax = 0u;
#pragma unroll
    for (int r = 0; r < 32; ++r) {
      umin = min(umin, k[r]);
      umax = max(umax, k[r]);
      kmin = min(kmin, key_from_bits(k[r]));
      kmax = max(kmax, key_from_bits(k[r]));
    }
    umin = __reduce_min_sync(0xffffffffu, umin);
    umax = __reduce_max_sync(0xffffffffu, umax);
    kmin = __reduce_min_sync(0xffffffffu, kmin);
    kmax = __reduce_max_sync(0xffffffffu, kmax);
    const bool raw = umin > 0u && umax < 0x7F800000u;
    const bool finite = kmin > 0x007FFFFFu && kmax < 0xFF800000u;
    const float vmin = __uint_as_float(bits_from_key(kmin));
    const float range = __fsub_rn(__uint_as_float(bits_from_key(kmax)), vmin);
    const float s = __fdiv_rn((float)GAS_BK_TOP, range);
    const bool ok = finite && range > 0.0f && range <= 3.402823466e38f && s <= 3.402823466e38f;
    const uint32_t mk = kl_mult(kmin, kmax);
#pragma unroll
    for (int j = 0; j < 6; ++j) h[lane + 32 * j] = 0u;
    __syncwarp();
    if (ok) {
#pragma unroll
      for (int r = 0; r < 32; ++r)
        if (cw_valid<VEC>(r, lane, n)) atomicAdd(&h[bucket_bits(k[r], vmin, s) - 0x4B000000u], 1u);
    }
    __syncwarp();
    const bool vfit = ok && __reduce_max_sync(0xffffffffu, max(h[lane], h[lane + 32])) <= 32u;
    bool kfit = false;  // counted only when the value buckets do not fit (the sampler is on the critical path)
    if (VEC && !vfit) {
#pragma unroll
      for (int r = 0; r < 32; ++r)
        if (cw_valid<VEC>(r, lane, n)) atomicAdd(&h[64u + __umulhi(key_from_bits(k[r]) - kmin, mk)], 1u);
      __syncwarp();
      kfit = __reduce_max_sync(0xffffffffu, max(h[64 + lane], h[96 + lane])) <= 32u;
    }
    const uint32_t k0 = bk_sample_key<VEC>(k, lane);
    const bool special = !raw && s1_sample_special(k0) >= 2;
    const bool to_split = special || (ok && bk_sample_dup(k0, vmin, s));
    if (lane == 0) {
      if (vfit) atomicAdd(&votes[0], 1u);
      if (kfit) atomicAdd(&votes[1], 1u);
      atomicAdd(&votes[to_split ? 3 : 2], 1u);
      if (special) atomicAdd(&votes[5], 1u);
    }
  }
  __syncthreads();
  uint32_t best = kS1Count;
  if ((int64_t)votes[0] * 32 >= 26 * S) best = kS1Bucket;
  else if ((int64_t)votes[1] * 32 >= 27 * S) best = kS1KeyLin;
  if (force <= kS1Cdf) best = force;
  // ---- 2. (only when neither map fits, or forced) the batch-CDF table from all
  // sampled keys, then each sampled array's bucket sizes under it (block-uniform branch)
  const bool want_cdf = force <= kS1Cdf ? force == kS1Cdf : (best == kS1Count && VEC);
  if (want_cdf) {
    if (active) {
#pragma unroll
      for (int r = 0; r < 32; ++r)
        if (cw_valid<VEC>(r, lane, n)) atomicAdd(&h512[key_from_bits(k[r]) >> 23], 1u);
    }
    __syncthreads();
    // exclusive scan of the 512 bins (16 warps), then (A_e, B_e) of cdf_bucket_addr
    uint32_t cnt = 0, total = 0;
    if (threadIdx.x < kCdfEntries) {
      cnt = h512[threadIdx.x];
      uint32_t x = cnt;
#pragma unroll
      for (int m = 1; m < 32; m <<= 1) {
        const uint32_t y = __shfl_up_sync(0xffffffffu, x, m);
        if (lane >= m) x += y;
      }
      if (lane == 31) part[w] = x;
      h512[threadIdx.x] = x - cnt;  // exclusive prefix inside the warp
    }
    __syncthreads();
    if (threadIdx.x < kCdfEntries) {
      uint32_t before = 0;
#pragma unroll
      for (int i = 0; i < kCdfEntries / 32; ++i) {
        before += i < w ? part[i] : 0u;
        total += part[i];
      }
      const uint64_t P = before + h512[threadIdx.x], T = total ? total : 1u;
      const uint64_t A = (P << 32) / T;
      const uint2 e = make_uint2(A > 0xFFFFFFFFull ? 0xFFFFFFFFu : (uint32_t)A, (uint32_t)(((uint64_t)cnt << 16) / T));
      tbl[threadIdx.x] = e;
      ctl->cdf[threadIdx.x] = e;
    }
    __syncthreads();
    if (active) {
      const uint32_t tsa = (uint32_t)__cvta_generic_to_shared(tbl);
#pragma unroll
      for (int r = 0; r < 32; ++r)
        if (cw_valid<VEC>(r, lane, n)) atomicAdd(&h[128u + (cdf_bucket_addr(key_from_bits(k[r]), tsa, 0u) >> 2)], 1u);
      __syncwarp();
      const bool cfit = __reduce_max_sync(0xffffffffu, max(h[128 + lane], h[160 + lane])) <= 32u;
      if (lane == 0 && cfit) atomicAdd(&votes[4], 1u);
    }
    __syncthreads();
    if (force > kS1Cdf && (int64_t)votes[4] * 32 >= 27 * S) best = kS1Cdf;
  }
  if (threadIdx.x == 0) {
    if (force > kS1Cdf && best == kS1Count) best = votes[3] > votes[2] ? kS1Split : kS1Count;
    ctl->flag = (!VEC && (best == kS1KeyLin || best == kS1Cdf)) ? kS1Count : best;  // those kernels take 16-byte rows only
    ctl->nlist = 0;
    ctl->split_kind = 2 * votes[5] > votes[3] ? kSplitSpecial : kSplitDup;
  }
}

// Loads array a (raw bits; slots past the end are copies of k[0]).
template <bool VEC>
__device__ __forceinline__ void s1_load(uint32_t (&k)[32], const uint32_t* arr, int n, int lane) {
  if constexpr (VEC) {
    const uint4* src = reinterpret_cast<const uint4*>(arr);
    const int nc = n >> 2;
#pragma unroll
    for (int q = 0; q < 8; ++q) {
      const int c = lane + 32 * q;
      const uint4 v = q < 4 ? ld_stream(src + c) : ldg_cs_if(c < nc, src + c);
      k[4 * q] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
    }
  } else {
#pragma unroll
    for (int r = 0; r < 32; ++r) k[r] = cw_valid<VEC>(r, lane, n) ? ld_stream(arr + lane + 32 * r) : 0u;
  }
#pragma unroll
  for (int r = 16; r < 32; ++r) k[r] = cw_valid<VEC>(r, lane, n) ? k[r] : k[0];
}

// 3. The counting sort (cw1024.cuh) over the whole batch (flag == count).
template <bool VEC>
__global__ void __launch_bounds__(kCwBlock, 1) k_s1_count(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one,
                                                          S1Ctl* ctl) {
  extern __shared__ __align__(16) uint4 cw_smem[];
  if (ctl->flag != kS1Count) return;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const uint32_t cnt_sa = (uint32_t)__cvta_generic_to_shared(cw_smem) + warp * kCwWarpBytes;
  const uint32_t buf_sa = cnt_sa + kCwCntBytes;
  uint32_t* const buf_ptr =
      reinterpret_cast<uint32_t*>(reinterpret_cast<unsigned char*>(cw_smem) + warp * kCwWarpBytes + kCwCntBytes);
  const int64_t nwarps = (int64_t)gridDim.x * (kCwBlock / 32);
  for (int64_t a = (int64_t)blockIdx.x * (kCwBlock / 32) + warp; a < N; a += nwarps) {
    uint32_t* const arr = d + a * (int64_t)n;
    uint32_t k[32];
    s1_load<VEC>(k, arr, n, lane);
#if GAS_BK_PREFETCH
    prefetch_l2_elect(a + nwarps < N, d + (a + nwarps) * (int64_t)n, n);
#endif
    uint32_t umin = k[0], umax = k[0];
#pragma unroll
    for (int r = 1; r < 31; r += 2) {
      umin = __vimin3_u32(umin, k[r], k[r + 1]);
      umax = __vimax3_u32(umax, k[r], k[r + 1]);
    }
    umin = __reduce_min_sync(0xffffffffu, min(umin, k[31]));
    umax = __reduce_max_sync(0xffffffffu, max(umax, k[31]));
    const bool raw = umin > 0u && umax < 0x7F800000u;
    if (!raw && s1_sample_special(bk_sample_key<VEC>(k, lane)) >= 2) {
      s1_push(ctl->nlist, s1_list(ctl), a, lane);  // special-heavy: the split kernel takes it
      continue;
    }
    cw_sort_warp<VEC>(k, raw, umin, umax, 0u, arr, n, lane, cnt_sa, buf_sa, buf_ptr, one);
  }
}

}  // namespace gas
