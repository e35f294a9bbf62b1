// cluster_sort.cuh — arrays longer than one CTA can hold (16384 < n <= 65536,
// SURVEY.md §8(f) row f4): one thread-block cluster of 8 CTAs per array.
//
// The paper designs for spectra of <= ~4000 peaks and sorts each
// array inside one block; past one SM's registers and shared
// memory the array is split by VALUE across the SMs of a cluster, the paper's
// own bucket idea (§4.1) one level up:
//  1. CTA c loads its slice [c n/8, (c+1) n/8) (16 keys per thread) and its
//     key min / max; the cluster's min / max come from the 8 CTAs' shared
//     memory over DSMEM;
//  2. each CTA counts its keys into 1024 key-linear coarse bins
//     f = (key - kmin) >> sh; every CTA then reads all 8 histograms over DSMEM
//     (8 x 4 KB) and derives the same partition: part p = the bins whose
//     exclusive prefix lies in [p n/8, (p+1) n/8) (monotone in the key), its
//     array positions [start_p, start_{p+1}) and this CTA's write offset in it;
//  3. each CTA writes its keys into their parts' positions of the array itself
//     (through L2: the whole cluster's 256 KB stay resident), then a cluster
//     barrier;
//  4. CTA p sorts part p in place with the CTA bucket sort of bucket_cta.cuh
//     (the size class of the part's length, on a named barrier over the warps
//     it needs). Parts are value ranges in order, so the array is sorted.
// A part longer than 16384 keys (a coarse bin holding > 1/8 of the array) is
// left as is and the array goes to a list; k_cluster_fallback then sorts those
// arrays with a global-memory bitonic network (slow, rare, always correct: the
// array is a permutation of its input at every step).
#pragma once
#include <cstdint>
#include <cooperative_groups.h>

#include "bucket_cta.cuh"

namespace gas {

namespace cgx = cooperative_groups;

constexpr int kClC = 8;                  // CTAs per cluster (portable maximum)
constexpr int kClT = 512;                // threads per CTA
constexpr int kClKeys = 16;              // keys per thread in step 1
constexpr int kClBins = 1024;            // coarse bins
constexpr int kClMaxLen = kClC * kClT * kClKeys;  // 65536
constexpr int kClPartMax = 16384;        // BkCta<16, 16> capacity
constexpr int kClSmem = BkCta<16, 16>::SMEM;

// The part sort: the CTA bucket sort of the part's size class, run by the
// first WR warps (named barrier 1 over them; the other warps skip it).
template <int W, int WR, int RV = 16>
__device__ __forceinline__ void cl_part_sort(uint32_t* arr, int len, unsigned char* sm, uint32_t one, int t) {
  if (t < 32 * WR) bucket_sort_cta<W, WR, false, RV>(arr, len, sm, one, t, 1u | ((uint32_t)(32 * WR) << 8));
}

// Parts of <= 256 keys: the first warp sorts them with the 1024-key network.
__device__ __forceinline__ void cl_small_sort(uint32_t* arr, int len, unsigned char* sm, uint32_t one, int t) {
  if (t >= 32) return;
  if (GAS_BKC_TMA_STORE && t == 0) asm volatile("cp.async.bulk.wait_group.read 0;" ::: "memory");  // sm is scratch here
  __syncwarp();
  uint32_t k[32];
#pragma unroll
  for (int r = 0; r < 32; ++r) {
    const int e = t * 32 + r;
    k[r] = e < len ? key_from_bits(arr[e]) : kPadKey;
  }
  sort1024_warp(k, t, reinterpret_cast<uint32_t*>(sm), one);
#pragma unroll
  for (int r = 0; r < 32; ++r) {
    const int e = t * 32 + r;
    if (e < len) arr[e] = bits_from_key(k[r]);
  }
  __syncwarp();
}

__device__ __forceinline__ void cl_sort_part(uint32_t* arr, int len, unsigned char* sm, uint32_t one, int t) {
  if (len <= 1) return;
  if (len > 8192) cl_part_sort<16, 16>(arr, len, sm, one, t);
  else if (len > 4096) cl_part_sort<8, 8>(arr, len, sm, one, t);
  else if (len > 2048) cl_part_sort<4, 4>(arr, len, sm, one, t);
  else if (len > 1024) cl_part_sort<2, 2>(arr, len, sm, one, t);
  else if (len > 512) cl_part_sort<1, 1>(arr, len, sm, one, t);
  else if (len > 256) cl_part_sort<1, 1, 8>(arr, len, sm, one, t);
  else cl_small_sort(arr, len, sm, one, t);
}

// One cluster per array (persistent over arrays); `fail` (count, then indices)
// receives the arrays with a part longer than kClPartMax.
__global__ void __cluster_dims__(kClC, 1, 1) __launch_bounds__(kClT, 1)
    k_cluster_sort(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one, uint32_t* __restrict__ fail) {
  extern __shared__ __align__(16) unsigned char cl_smem[];
  __shared__ uint32_t hist[kClBins];     // this CTA's coarse histogram (read by the peers)
  __shared__ unsigned char bpart[kClBins];
  __shared__ uint32_t red[2 * (kClT / 32)];
  __shared__ uint32_t kmm[2];            // this CTA's key min / max (read by the peers)
  __shared__ uint32_t scan[kClT / 32];
  __shared__ uint32_t pstart[kClC + 1];  // part p = array positions [pstart[p], pstart[p+1])
  __shared__ uint32_t pbase[kClC];       // this CTA's first position in part p
  __shared__ uint32_t pcnt[kClC];        // keys of this CTA written to part p so far
  cgx::cluster_group cl = cgx::this_cluster();
  const int c = (int)cl.block_rank();
  const int t = threadIdx.x, lane = t & 31, warp = t >> 5;
  const int64_t nclusters = gridDim.x / kClC, cid = blockIdx.x / kClC;
  for (int64_t a = cid; a < N; a += nclusters) {
    uint32_t* const arr = d + a * (int64_t)n;
    const int s0 = (int)(((int64_t)c * n) / kClC), s1 = (int)(((int64_t)(c + 1) * n) / kClC), sl = s1 - s0;
    // ---- 1. load this CTA's slice as ordered keys; CTA min / max
    uint32_t k[kClKeys];
    uint32_t kmin = 0xFFFFFFFFu, kmax = 0u;
#pragma unroll
    for (int r = 0; r < kClKeys; ++r) {
      const int e = t + kClT * r;
      k[r] = e < sl ? key_from_bits(__ldcg(arr + s0 + e)) : 0u;  // L2 only: peers rewrite these lines in step 3
      if (e < sl) { kmin = min(kmin, k[r]); kmax = max(kmax, k[r]); }
    }
    kmin = __reduce_min_sync(0xffffffffu, kmin);
    kmax = __reduce_max_sync(0xffffffffu, kmax);
    if (lane == 0) { red[2 * warp] = kmin; red[2 * warp + 1] = kmax; }
    for (int b = t; b < kClBins; b += kClT) hist[b] = 0u;
    if (t < kClC) pcnt[t] = 0u;
    __syncthreads();
    if (t == 0) {
      uint32_t lo = 0xFFFFFFFFu, hi = 0u;
      for (int w = 0; w < kClT / 32; ++w) { lo = min(lo, red[2 * w]); hi = max(hi, red[2 * w + 1]); }
      kmm[0] = lo;
      kmm[1] = hi;
    }
    cl.sync();  // every CTA's kmm is final
    kmin = 0xFFFFFFFFu;
    kmax = 0u;
#pragma unroll
    for (int r = 0; r < kClC; ++r) {
      const uint32_t* p = cl.map_shared_rank(kmm, r);
      kmin = min(kmin, p[0]);
      kmax = max(kmax, p[1]);
    }
    const int bits = 32 - __clz(kmax - kmin);
    const uint32_t sh = bits > 10 ? (uint32_t)(bits - 10) : 0u;
    // ---- 2. coarse histogram, then the partition from all 8 histograms
#pragma unroll
    for (int r = 0; r < kClKeys; ++r)
      if (t + kClT * r < sl) atomicAdd(&hist[(k[r] - kmin) >> sh], 1u);
    cl.sync();  // every CTA's histogram is final
    // thread t owns bins 2t, 2t + 1: total count g and the count in lower CTAs
    uint32_t g[2], pre[2];
#pragma unroll
    for (int j = 0; j < 2; ++j) {
      g[j] = 0u;
      pre[j] = 0u;
    }
#pragma unroll
    for (int r = 0; r < kClC; ++r) {
      const uint32_t* h = cl.map_shared_rank(hist, r);
#pragma unroll
      for (int j = 0; j < 2; ++j) {
        const uint32_t v = h[2 * t + j];
        g[j] += v;
        pre[j] += r < c ? v : 0u;
      }
    }
    // exclusive scan of g over the bins (warp scan + scan of the warp totals)
    uint32_t x = g[0] + g[1];
#pragma unroll
    for (int m = 1; m < 32; m <<= 1) {
      const uint32_t y = __shfl_up_sync(0xffffffffu, x, m);
      if (lane >= m) x += y;
    }
    if (lane == 31) scan[warp] = x;
    __syncthreads();
    uint32_t wbase = 0;
    for (int w = 0; w < warp; ++w) wbase += scan[w];
    const uint32_t cum0 = wbase + x - g[0] - g[1], cum1 = cum0 + g[0];  // prefix before bins 2t, 2t + 1
    const int p0 = min((int)((uint64_t)cum0 * kClC / (uint64_t)n), kClC - 1);
    const int p1 = min((int)((uint64_t)cum1 * kClC / (uint64_t)n), kClC - 1);
    bpart[2 * t] = (unsigned char)p0;
    bpart[2 * t + 1] = (unsigned char)p1;
    if (t == 0) {
      pstart[0] = 0u;
      pstart[kClC] = (uint32_t)n;
    }
    if (t < kClC) pbase[t] = 0u;
    __syncthreads();
    // part p starts at the prefix of its first bin; parts with no bin are empty
    {
      const int pp = t == 0 ? -1 : (int)bpart[2 * t - 1];
      for (int p = pp + 1; p <= p0; ++p) if (p > 0) pstart[p] = cum0;
      for (int p = p0 + 1; p <= p1; ++p) pstart[p] = cum1;
      if (t == kClT - 1)
        for (int p = p1 + 1; p < kClC; ++p) pstart[p] = (uint32_t)n;
    }
    // this CTA's offset inside each part: keys of that part in lower CTAs
    if (pre[0]) atomicAdd(&pbase[p0], pre[0]);
    if (pre[1]) atomicAdd(&pbase[p1], pre[1]);
    __syncthreads();
    // ---- 3. write the keys (as bits) to their part positions of the array
#pragma unroll
    for (int r = 0; r < kClKeys; ++r) {
      if (t + kClT * r < sl) {
        const int p = bpart[(k[r] - kmin) >> sh];
        const uint32_t pos = pstart[p] + pbase[p] + atomicAdd(&pcnt[p], 1u);
        arr[pos] = bits_from_key(k[r]);
      }
    }
    __threadfence();
    cl.sync();  // every part is complete in memory (and no peer still reads this CTA's hist / kmm)
    // ---- 4. sort part c in place
    const int plo = (int)pstart[c], plen = (int)pstart[c + 1] - plo;
    if (c == 0 && t == 0) {  // every CTA holds the same pstart: CTA 0 lists the array once
      bool over = false;
      for (int p = 0; p < kClC; ++p) over |= pstart[p + 1] - pstart[p] > (uint32_t)kClPartMax;
      if (over) fail[1 + atomicAdd(&fail[0], 1u)] = (uint32_t)a;
    }
    if (plen <= kClPartMax) cl_sort_part(arr + plo, plen, cl_smem, one, t);
    __syncthreads();
  }
  if (GAS_BKC_TMA_STORE && t == 0) asm volatile("cp.async.bulk.wait_group 0;" ::: "memory");  // part stores complete
}

// The rare arrays with an oversize part: a global-memory bitonic network over
// the padded power-of-two length (virtual elements are +max keys), one CTA of
// 1024 threads per array.
__global__ void __launch_bounds__(1024, 1) k_cluster_fallback(uint32_t* __restrict__ d, int n, const uint32_t* fail) {
  const uint32_t cnt = fail[0];
  int P = 1;
  while (P < n) P <<= 1;
  for (uint32_t i = blockIdx.x; i < cnt; i += gridDim.x) {
    uint32_t* const arr = d + (int64_t)fail[1 + i] * n;
    for (int e = threadIdx.x; e < n; e += blockDim.x) arr[e] = key_from_bits(arr[e]);
    __syncthreads();
    // mirror form of bitonic sort (bitonic.cuh): every compare-exchange puts the
    // minimum at the lower index, so the virtual +max elements past n never move
    for (int kk = 2; kk <= P; kk <<= 1) {
      for (int j = kk >> 1; j > 0; j >>= 1) {
        const int m = j == (kk >> 1) ? kk - 1 : j;  // first stage of a merge: the mirror partner
        for (int x = threadIdx.x; x < P; x += blockDim.x) {
          const int y = x ^ m;
          if (y > x && y < n) {
            const uint32_t a = arr[x], b = arr[y];
            if (a > b) { arr[x] = b; arr[y] = a; }
          }
        }
        __syncthreads();
      }
    }
    for (int e = threadIdx.x; e < n; e += blockDim.x) arr[e] = bits_from_key(arr[e]);
    __syncthreads();
  }
}

}  // namespace gas
