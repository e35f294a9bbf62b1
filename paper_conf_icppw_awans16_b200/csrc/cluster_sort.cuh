// cluster_sort.cuh — arrays longer than one CTA can hold (16384 < n <= 65536,
// SURVEY.md §8(f) row f4): one thread-block cluster of C = 8 or 16 CTAs per array.
//
// The paper designs for spectra of <= ~4000 peaks and sorts each
// array inside one block; past one SM's registers and shared
// memory the array is split by VALUE across the SMs of a cluster, the paper's
// own bucket idea (§4.1) one level up:
//  1. CTA c loads its slice [c n/C, (c+1) n/C) and its key min / max; the
//     cluster's min / max come from the C CTAs' shared memory over DSMEM;
//  2. each CTA counts its keys into 256 coarse bins (value-linear over the
//     array's range when every value is finite, else key-linear
//     f = (key - kmin) >> sh); every CTA then reads all C histograms over DSMEM
//     and derives the same partition: part p = the bins whose exclusive prefix
//     lies in [p n/C, (p+1) n/C) (monotone in the key), its array positions
//     [start_p, start_{p+1}) and this CTA's write offset in it;
//  3. each CTA writes its keys into their parts' positions of the array itself
//     (through L2: the cluster's array stays resident), then a cluster barrier;
//  4. CTA p sorts part p in place with the CTA bucket sort of bucket_cta.cuh
//     (the CTA's own class when the part fills it, else the class of the
//     part's length on the first warps). Parts are value ranges in order, so
//     the array is sorted.
// A part longer than the CTA class holds (a coarse bin holding a large share
// of the array) is left as is and the array goes to a list; k_cluster_fallback
// then sorts those arrays with a global-memory bitonic network (slow, rare,
// always correct: the array is a permutation of its input at every step).
#pragma once
#include <cstdint>
#include <cooperative_groups.h>

#include "bucket_cta.cuh"

namespace gas {

namespace cgx = cooperative_groups;

// Cluster configurations (round 2): CTAs sized to their part. Round 1 used 8
// CTAs of 512 threads (150 KB of shared memory, one per SM) per array, so an
// SM held one array's part of 2-8 K keys sorted by the 2-8 warps of its class:
// 0.03-0.06 of the HBM roofline. Here a CTA has exactly the WR warps of its
// part's class and that class's shared memory, C CTAs per cluster (8, or 16
// non-portable) keep each part at 2-4 K keys, and several clusters share an SM
// (4-5 CTAs per SM, 20 warps).
//   C = 8, <4, 4>:   16384 < n <= 24576 (parts ~2048-3072 of 4096)
//   C = 8, <8, 5>:   24576 < n <= 32768 (parts ~3072-4096 of 5120)
//   C = 8, <16, 12>: 32768 < n <= 65536 (parts ~4096-8192 of 12288; one CTA per SM)
// (Measured: non-portable 16-CTA clusters of <4,4> / <8,5> CTAs for n > 32768
// ran 2-4x slower than these.)
template <int W, int WR, int C, int MAXN>
struct ClCfg {
  static constexpr int T = 32 * WR;                     // threads per CTA
  static constexpr int KPT1 = (MAXN + C * T - 1) / (C * T);  // keys per thread in step 1
  static constexpr int NB2 = 128;                       // threads owning coarse bins (2 each)
  static constexpr int NB = 2 * NB2;                    // coarse bins
  static constexpr int CAP = 1024 * WR;                 // part capacity (the CTA class)
  static constexpr int SMEM = BkCta<W, WR>::SMEM;
  static_assert(T >= NB2, "bin owners");
};
constexpr int kClMaxLen = 65536;

// The part sort: the CTA bucket sort of the part's size class, run by the
// first WR' warps of the CTA (named barrier 1 over them; the other warps skip it).
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

// Part of len <= CAP keys: all WR warps when it fills more than 16 keys per
// thread, else the standard class of its length on the first warps.
template <int W, int WR>
__device__ __forceinline__ void cl_sort_part(uint32_t* arr, int len, unsigned char* sm, uint32_t one, int t) {
  constexpr int T = 32 * WR;
  if (len <= 1) return;
  if (len > 16 * T) cl_part_sort<W, WR, 16>(arr, len, sm, one, t);
  else if (WR > 6 && len > 4096) cl_part_sort<8, 6>(arr, len, sm, one, t);
  else if (WR > 4 && len > 3072) cl_part_sort<4, 4>(arr, len, sm, one, t);
  else if (WR > 3 && len > 2048) cl_part_sort<4, 3>(arr, len, sm, one, t);
  else if (len > 1024) cl_part_sort<2, 2>(arr, len, sm, one, t);
  else if (len > 512) cl_part_sort<1, 1>(arr, len, sm, one, t);
  else if (len > 256) cl_part_sort<1, 1, 8>(arr, len, sm, one, t);
  else cl_small_sort(arr, len, sm, one, t);
}

// One cluster of C CTAs per array (persistent over arrays; the cluster shape
// is a launch attribute); `fail` (count, then indices) receives the arrays
// with a part longer than the CTA class holds.
// PART (the two-kernel path, cluster_partition_sort): steps 1-3 only; CTA 0
// writes the C part boundaries of array a to parts[a C .. a C + C - 1]
// (element offsets into the batch: a CSR of N C parts) and lists the array in
// `fail` when a part exceeds kClPartMaxOff; no dynamic shared memory.
constexpr int kClPartMaxOff = 16384;  // longest part the offsets classes take
template <int W, int WR, int C, int MAXN, bool PART = false>
__global__ void __launch_bounds__(32 * WR, PART ? 3 : bkc_min_blocks<WR>())
    k_cluster_sort(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one, uint32_t* __restrict__ fail,
                   int64_t* __restrict__ parts) {
  using G = ClCfg<W, WR, C, MAXN>;
  constexpr int T = G::T, NB = G::NB, NB2 = G::NB2, KPT1 = G::KPT1;
  extern __shared__ __align__(16) unsigned char cl_smem[];
  __shared__ uint32_t hist[NB];          // this CTA's coarse histogram (read by the peers)
  __shared__ unsigned char bpart[NB];
  __shared__ uint32_t red[2 * WR];
  __shared__ uint32_t kmm[2];            // this CTA's key min / max (read by the peers)
  __shared__ uint32_t scan[NB2 / 32];
  __shared__ uint32_t pstart[C + 1];     // part p = array positions [pstart[p], pstart[p+1])
  __shared__ uint32_t binpos[NB];        // next array position of this CTA's keys of bin b (atomic)
  cgx::cluster_group cl = cgx::this_cluster();
  const int c = (int)cl.block_rank();
  const int t = threadIdx.x, lane = t & 31, warp = t >> 5;
  const int64_t nclusters = gridDim.x / C, cid = blockIdx.x / C;
  for (int64_t a = cid; a < N; a += nclusters) {
    uint32_t* const arr = d + a * (int64_t)n;
    const int s0 = (int)(((int64_t)c * n) / C), s1 = (int)(((int64_t)(c + 1) * n) / C), sl = s1 - s0;
    // ---- 1. load this CTA's slice as ordered keys; CTA min / max
    uint32_t k[KPT1];
    uint32_t kmin = 0xFFFFFFFFu, kmax = 0u;
#pragma unroll
    for (int r = 0; r < KPT1; ++r) {
      const int e = t + T * r;
      k[r] = e < sl ? key_from_bits(__ldcg(arr + s0 + e)) : 0u;  // L2 only: peers rewrite these lines in step 3
      if (e < sl) { kmin = min(kmin, k[r]); kmax = max(kmax, k[r]); }
    }
    kmin = __reduce_min_sync(0xffffffffu, kmin);
    kmax = __reduce_max_sync(0xffffffffu, kmax);
    if (lane == 0) { red[2 * warp] = kmin; red[2 * warp + 1] = kmax; }
    for (int b = t; b < NB; b += T) hist[b] = 0u;
    __syncthreads();
    if (t == 0) {
      uint32_t lo = 0xFFFFFFFFu, hi = 0u;
      for (int w = 0; w < WR; ++w) { lo = min(lo, red[2 * w]); hi = max(hi, red[2 * w + 1]); }
      kmm[0] = lo;
      kmm[1] = hi;
    }
    cl.sync();  // every CTA's kmm is final
    kmin = 0xFFFFFFFFu;
    kmax = 0u;
#pragma unroll
    for (int r = 0; r < C; ++r) {
      const uint32_t* p = cl.map_shared_rank(kmm, r);
      kmin = min(kmin, p[0]);
      kmax = max(kmax, p[1]);
    }
    const int bits = 32 - __clz(kmax - kmin);
    constexpr int LNB = NB == 256 ? 8 : 9;
    const uint32_t sh = bits > LNB ? (uint32_t)(bits - LNB) : 0u;
    // coarse bin of a key: value-linear over [vmin, vmax] when every value is
    // finite (the map of bucket1024.cuh: uniform values give uniform bins, and
    // few lanes of a warp hit one counter), else key-linear; both monotone
    const float vmin = __uint_as_float(bits_from_key(kmin));
    const float vrange = __fsub_rn(__uint_as_float(bits_from_key(kmax)), vmin);
    const float vs = __fdiv_rn((float)(NB - 1), vrange);
    const bool vmap = kmin > 0x007FFFFFu && kmax < 0xFF800000u && vrange > 0.0f && vrange <= 3.402823466e38f &&
                      vs <= 3.402823466e38f;
    auto bin = [&](uint32_t kk) -> uint32_t {
      return vmap ? bucket_bits(bits_from_key(kk), vmin, vs) - 0x4B000000u : (kk - kmin) >> sh;
    };
    // ---- 2. coarse histogram, then the partition from all C histograms
#pragma unroll
    for (int r = 0; r < KPT1; ++r)
      if (t + T * r < sl) atomicAdd(&hist[bin(k[r])], 1u);
    cl.sync();  // every CTA's histogram is final
    // thread t < NB2 owns bins 2t, 2t + 1: total count g and the count in lower CTAs
    uint32_t g[2] = {0u, 0u}, pre[2] = {0u, 0u};
    if (t < NB2) {
#pragma unroll
      for (int r = 0; r < C; ++r) {
        const uint32_t* hr = cl.map_shared_rank(hist, r);
#pragma unroll
        for (int j = 0; j < 2; ++j) {
          const uint32_t v = hr[2 * t + j];
          g[j] += v;
          pre[j] += r < c ? v : 0u;
        }
      }
    }
    // exclusive scan of g over the bins (warp scan + scan of the warp totals)
    uint32_t x = g[0] + g[1];
#pragma unroll
    for (int m = 1; m < 32; m <<= 1) {
      const uint32_t y = __shfl_up_sync(0xffffffffu, x, m);
      if (lane >= m) x += y;
    }
    if (lane == 31 && t < NB2) scan[warp] = x;
    __syncthreads();
    int p0 = 0, p1 = 0;
    uint32_t cum0 = 0, cum1 = 0;
    if (t < NB2) {
      uint32_t wbase = 0;
      for (int w = 0; w < warp; ++w) wbase += scan[w];
      cum0 = wbase + x - g[0] - g[1];  // prefix before bins 2t, 2t + 1
      cum1 = cum0 + g[0];
      p0 = min((int)((uint64_t)cum0 * C / (uint64_t)n), C - 1);
      p1 = min((int)((uint64_t)cum1 * C / (uint64_t)n), C - 1);
      bpart[2 * t] = (unsigned char)p0;
      bpart[2 * t + 1] = (unsigned char)p1;
    }
    if (t == 0) {
      pstart[0] = 0u;
      pstart[C] = (uint32_t)n;
    }
    __syncthreads();
    if (t < NB2) {
      // part p starts at the prefix of its first bin; parts with no bin are empty
      const int pp = t == 0 ? -1 : (int)bpart[2 * t - 1];
      for (int p = pp + 1; p <= p0; ++p) if (p > 0) pstart[p] = cum0;
      for (int p = p0 + 1; p <= p1; ++p) pstart[p] = cum1;
      if (t == NB2 - 1)
        for (int p = p1 + 1; p < C; ++p) pstart[p] = (uint32_t)n;
      // bins are laid out in key order over the whole array: this CTA's keys of
      // bin b start at the prefix of b plus the keys of b in lower CTAs
      binpos[2 * t] = cum0 + pre[0];
      binpos[2 * t + 1] = cum1 + pre[1];
    }
    __syncthreads();
    // ---- 3. write the keys (as bits) to their part positions of the array
#pragma unroll
    for (int r = 0; r < KPT1; ++r) {
      if (t + T * r < sl) {
        const uint32_t pos = atomicAdd(&binpos[bin(k[r])], 1u);
        arr[pos] = bits_from_key(k[r]);
      }
    }
    cl.sync();  // every part is complete in memory (barrier.cluster arrive.release / wait.acquire) (and no peer still reads this CTA's hist / kmm)
    if constexpr (PART) {
      if (c == 0 && t < C) parts[a * C + t] = a * (int64_t)n + pstart[t];
      if (c == 0 && t == 0) {
        bool over = false;
        for (int p = 0; p < C; ++p) over |= pstart[p + 1] - pstart[p] > (uint32_t)kClPartMaxOff;
        if (over) fail[1 + atomicAdd(&fail[0], 1u)] = (uint32_t)a;
      }
      __syncthreads();  // pstart is rewritten by the next array
    } else {
      // ---- 4. sort part c in place
      const int plo = (int)pstart[c], plen = (int)pstart[c + 1] - plo;
      if (c == 0 && t == 0) {  // every CTA holds the same pstart: CTA 0 lists the array once
        bool over = false;
        for (int p = 0; p < C; ++p) over |= pstart[p + 1] - pstart[p] > (uint32_t)G::CAP;
        if (over) fail[1 + atomicAdd(&fail[0], 1u)] = (uint32_t)a;
      }
      if (plen <= G::CAP) cl_sort_part<W, WR>(arr + plo, plen, cl_smem, one, t);
      __syncthreads();
    }
  }
  if (PART && blockIdx.x == 0 && t == 0) parts[N * C] = N * (int64_t)n;  // the CSR's closing offset
  if (!PART && GAS_BKC_TMA_STORE && t == 0) asm volatile("cp.async.bulk.wait_group 0;" ::: "memory");  // part stores complete
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
