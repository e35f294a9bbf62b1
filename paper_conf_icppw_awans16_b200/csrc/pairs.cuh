// pairs.cuh — stable key + payload variant (BASELINE.json north_star
// "optional key+payload variant"; reading C-2).
//
// Stability is obtained the data-oblivious way: the network sorts 64-bit
// elements (ordered key << 32 | original position), so equal keys are
// ordered by position and the result is unique. Payloads are staged in shared
// memory and gathered by position after the sort; keys and payloads are
// written back in place through a rank-order staging buffer (coalesced).
// Algorithmic bytes: 16n per array (keys and payloads read and written once).
// `list` (or nullptr): sort only the arrays it names (count, then indices) —
// the leftovers of the bucket kernel of pairs1024.cuh.
#pragma once
#include <cstdint>

#include "bitonic.cuh"
#include "ordered_key.cuh"
#include "segsort.cuh"  // swz

namespace gas {

template <int KPT, int G, int W>
struct PairsCfg {
  static constexpr int P = KPT * G * W;
  static constexpr int TH = G * W;                           // threads per array
  static constexpr int TPB = (W == 1) ? 256 : 32 * W;        // threads per block
  static constexpr int GROUPS = TPB / TH;                    // arrays per block per round
  static constexpr int BYTES_PER_GROUP = P * 4 * 2 + (W > 1 ? P * 8 : 0);
  static constexpr int SMEM = GROUPS * BYTES_PER_GROUP;
};

template <int KPT, int G, int W>
__global__ void __launch_bounds__(PairsCfg<KPT, G, W>::TPB)
    k_pairs(uint32_t* __restrict__ keys, uint32_t* __restrict__ vals, int64_t N, int n,
            const uint32_t* __restrict__ list) {
  using C = PairsCfg<KPT, G, W>;
  constexpr int P = C::P, TH = C::TH;
  extern __shared__ __align__(16) unsigned char pairs_smem[];
  const int grp = threadIdx.x / TH;            // array slot inside the block
  const int t = threadIdx.x % TH;              // thread index inside the array's owners
  const int g = t & (G - 1);                   // lane inside the G-lane group (W == 1) / lane (W > 1)
  unsigned char* base = pairs_smem + grp * C::BYTES_PER_GROUP;
  uint32_t* vs = reinterpret_cast<uint32_t*>(base);           // payloads, input order
  uint4* ks = reinterpret_cast<uint4*>(base + P * 4);         // rank-order staging (swizzled chunks)
  uint64_t* xs = reinterpret_cast<uint64_t*>(base + P * 8);   // cross-warp exchange (W > 1)
  if (list) N = list[0];  // a worklist (pairs1024.cuh): count, then array indices
  for (int64_t a0 = (int64_t)blockIdx.x * C::GROUPS; a0 < N; a0 += (int64_t)gridDim.x * C::GROUPS) {
    const bool valid = a0 + grp < N;
    const int64_t a = !valid ? 0 : (list ? (int64_t)list[1 + a0 + grp] : a0 + grp);
    const int64_t off = (valid ? a : 0) * (int64_t)n;
    uint64_t k[KPT];
#pragma unroll
    for (int q = 0; q < KPT; ++q) {
      const int e = t + TH * q;  // element e goes to thread t, slot q
      const bool in = valid && e < n;
      const uint32_t kb = in ? keys[off + e] : 0u;
      vs[e] = in ? vals[off + e] : 0u;
      k[q] = in ? ((uint64_t)key_from_bits(kb) << 32) | (uint32_t)e : ~0ull - (uint64_t)(P - e);
    }
    if constexpr (W > 1) __syncthreads(); else __syncwarp();
    Bitonic<KPT, G, W, uint64_t>::sort(k, g, t, xs, 1u);
    // gather payloads by original position, then stage keys and payloads in rank order
    uint32_t v[KPT];
#pragma unroll
    for (int r = 0; r < KPT; ++r) {
      const uint32_t pos = (uint32_t)k[r];
      v[r] = pos < (uint32_t)n ? vs[pos] : 0u;
    }
    if constexpr (W > 1) __syncthreads(); else __syncwarp();
#pragma unroll
    for (int r = 0; r < KPT; ++r) {
      const int w = t * KPT + r;  // rank held in register r
      reinterpret_cast<uint32_t*>(ks)[swz(w >> 2) * 4 + (w & 3)] = bits_from_key((uint32_t)(k[r] >> 32));
      vs[swz(w >> 2) * 4 + (w & 3)] = v[r];
    }
    if constexpr (W > 1) __syncthreads(); else __syncwarp();
    if (valid) {
#pragma unroll
      for (int q = 0; q < KPT; ++q) {
        const int w = t + TH * q;
        if (w < n) {
          keys[off + w] = reinterpret_cast<const uint32_t*>(ks)[swz(w >> 2) * 4 + (w & 3)];
          vals[off + w] = vs[swz(w >> 2) * 4 + (w & 3)];
        }
      }
    }
    if constexpr (W > 1) __syncthreads(); else __syncwarp();
  }
}

}  // namespace gas
