// pairs1024.cuh — the stable key + payload variant (gas_sort_pairs, SURVEY.md
// §8(f) row f2, reading C-2) on the value-bucket design of bucket1024.cuh,
// for 512 < n <= 1024 with 16-byte-aligned key and payload rows.
//
// (m/z, intensity) pairs are the paper's use case. The pure 64-bit
// network of pairs.cuh costs ~26 compare-exchanges of (key, position) per key;
// here, as for keys alone, one warp splits the array into 64 value buckets
// whose concatenation is the sorted array (§4.1) and each lane
// sorts two buckets of <= 32 keys in registers. Stability: every bucket slot
// holds (key, original position) — equal keys always share a bucket, since the
// bucket map is a function of the value — and the bucket network orders pairs
// lexicographically, so equal keys come out in input order; the payloads are
// then gathered by position. Per array:
//  1. load the keys (8 x LDG.128 per lane); min / max; all positive finite
//     -> raw bits are the keys, else the totalOrder keys (ordered_key.cuh);
//  2. the atomic on the bucket's counter returns the key's slot address (as in
//     bucket1024.cuh); key and position are stored at that slot of the key
//     rows and of the parallel position rows;
//  3. two rounds per lane (bucket lane + 32, then lane): load 32 keys and 32
//     positions, 191-comparator odd-even network on the pairs, staged in
//     rank order (keys over the drained key rows 32..63, positions over the
//     drained position rows 32..63);
//  4. store: keys from the staging (coalesced 16-byte stores); payloads
//     gathered from the payload row by the staged positions (L1), all of them
//     before the first in-place store, then 16-byte stores.
// Arrays the bucket map cannot take (a NaN or an infinity, a bucket of more
// than 32 keys, a range that overflows) go to a list that the pairs network
// kernel (pairs.cuh) sorts afterwards. Algorithmic bytes: 16 n per array.
#pragma once
#include <cstdint>

#include "bucket1024.cuh"
#include "pairs.cuh"

namespace gas {

#ifndef GAS_PB_BLOCK
#define GAS_PB_BLOCK 384
#endif
constexpr int kPbBlock = GAS_PB_BLOCK;                         // 12 warps per SM (18.7 KB of shared memory each)
constexpr int kPbPosDelta = kBkSlotBytes;             // position rows follow the key rows
constexpr int kPbWarpBytes = kBkCntBytes + 2 * kBkSlotBytes;
constexpr int kPbSmemBytes = (kPbBlock / 32) * kPbWarpBytes;
static_assert(kPbSmemBytes <= 232448, "pairs bucket kernel: shared memory per SM");

// Compare-exchange of (key, position) pairs, ascending in lexicographic order.
__device__ __forceinline__ void ce_kp(uint32_t& ka, uint32_t& pa, uint32_t& kb, uint32_t& pb) {
  const uint64_t a = ((uint64_t)ka << 32) | pa, b = ((uint64_t)kb << 32) | pb;
  const bool sw = a > b;
  const uint32_t k0 = sw ? kb : ka, p0 = sw ? pb : pa, k1 = sw ? ka : kb, p1 = sw ? pa : pb;
  ka = k0; pa = p0; kb = k1; pb = p1;
}

__device__ __forceinline__ void sort32_kp(uint32_t (&k)[32], uint32_t (&p)[32]) {
  constexpr OddEvenTable<32> T{};
#pragma unroll
  for (int c = 0; c < OddEvenTable<32>::C; ++c) ce_kp(k[T.e[c].a], p[T.e[c].a], k[T.e[c].b], p[T.e[c].b]);
}

// `fail`: the arrays left to the network kernel (count, then indices).
__global__ void __launch_bounds__(kPbBlock, 1)
    k_pairs_bucket1024(uint32_t* __restrict__ keys, uint32_t* __restrict__ vals, int64_t N, int n,
                       uint32_t* __restrict__ fail) {
  extern __shared__ __align__(16) uint4 pb_smem[];
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const uint32_t wsa = (uint32_t)__cvta_generic_to_shared(pb_smem) + warp * kPbWarpBytes;
  const uint32_t cnt_sa = wsa;
  const uint32_t slot_sa = wsa + kBkCntBytes;
  const uint32_t kst_sa = slot_sa + kBkStageWord * 4;    // key staging (rank order) over key rows 32..63
  const uint32_t pst_sa = kst_sa + kPbPosDelta;          // position staging over position rows 32..63
  const uint32_t slot_last = slot_sa + kBkSlotBytes - 4;
  const int nc = n >> 2;
  const int64_t nwarps = (int64_t)gridDim.x * (kPbBlock / 32);
  const uint32_t cnt_b0 = cnt_sa - 0x4B000000u * 4u;
  const uint32_t row0 = slot_sa + lane * (kBkRowWords * 4);
  const uint32_t row1 = row0 + 32 * (kBkRowWords * 4);

  for (int64_t a = (int64_t)blockIdx.x * (kPbBlock / 32) + warp; a < N; a += nwarps) {
    uint4* const kdst = reinterpret_cast<uint4*>(keys + a * (int64_t)n);
    uint4* const vdst = reinterpret_cast<uint4*>(vals + a * (int64_t)n);
    uint32_t k[32];
#pragma unroll
    for (int q = 0; q < 8; ++q) {
      const int c = lane + 32 * q;
      const uint4 v = q < 4 ? ld_stream(kdst + c) : ldg_cs_if(c < nc, kdst + c);
      k[4 * q] = v.x; k[4 * q + 1] = v.y; k[4 * q + 2] = v.z; k[4 * q + 3] = v.w;
    }
#if GAS_BK_PREFETCH
    prefetch_l2_elect(a + nwarps < N, keys + (a + nwarps) * (int64_t)n, n);
    prefetch_l2_elect(a + nwarps < N, vals + (a + nwarps) * (int64_t)n, n);
#endif
#pragma unroll
    for (int q = 4; q < 8; ++q) {
      const bool v = lane + 32 * q < nc;
#pragma unroll
      for (int j = 0; j < 4; ++j) k[4 * q + j] = v ? k[4 * q + j] : k[0];
    }
    uint32_t umin = k[0], umax = k[0];
#pragma unroll
    for (int r = 1; r < 31; r += 2) {
      umin = __vimin3_u32(umin, k[r], k[r + 1]);
      umax = __vimax3_u32(umax, k[r], k[r + 1]);
    }
    umin = __reduce_min_sync(0xffffffffu, min(umin, k[31]));
    umax = __reduce_max_sync(0xffffffffu, max(umax, k[31]));
    const bool raw = umin > 0u && umax < 0x7F800000u;
    bool use = true;
    if (!raw) {
      uint32_t kmin = 0xFFFFFFFFu, kmax = 0u;
#pragma unroll
      for (int r = 0; r < 32; ++r) {
        const uint32_t kk = key_from_bits(k[r]);
        kmin = min(kmin, kk);
        kmax = max(kmax, kk);
        k[r] = kk;
      }
      kmin = __reduce_min_sync(0xffffffffu, kmin);
      kmax = __reduce_max_sync(0xffffffffu, kmax);
      use = kmin > 0x007FFFFFu && kmax < 0xFF800000u;
      umin = bits_from_key(kmin);
      umax = bits_from_key(kmax);
    }
    const float vmin = __uint_as_float(umin), vmax = __uint_as_float(umax);
    const float range = __fsub_rn(vmax, vmin);
    const float s = __fdiv_rn((float)GAS_BK_TOP, range);
    use = use && range > 0.0f && range <= 3.402823466e38f && s <= 3.402823466e38f;
    uint32_t t0 = 0, t1 = 0, base0 = 0, base1 = 0;
    if (use) {
      sts32(cnt_sa + lane * 4, row0);
      sts32(cnt_sa + 128 + lane * 4, row1);
      __syncwarp();
      // key r of the lane is element 4 (lane + 32 (r >> 2)) + (r & 3); for non-raw arrays k holds
      // the keys, whose float value is bits_from_key(k)
#pragma unroll
      for (int g = 0; g < 32; g += 4) {
        uint32_t sa[4];
#pragma unroll
        for (int r = g; r < g + 4; ++r) {
          const uint32_t vb = raw ? k[r] : bits_from_key(k[r]);
          sa[r - g] = atoms_add4_if((r >> 2) < 4 || lane + 32 * (r >> 2) < nc, bucket_bits(vb, vmin, s) * 4u + cnt_b0);
        }
#pragma unroll
        for (int r = g; r < g + 4; ++r) {
          const bool v = (r >> 2) < 4 || lane + 32 * (r >> 2) < nc;
          const uint32_t at = min(sa[r - g], slot_last);
          sts32_if(v, at, k[r]);
          sts32_if(v, at + kPbPosDelta, 4u * (lane + 32u * (r >> 2)) + (r & 3));
        }
      }
      __syncwarp();
      t0 = (lds32(cnt_sa + lane * 4) - row0) >> 2;
      t1 = (lds32(cnt_sa + 128 + lane * 4) - row1) >> 2;
      use = __all_sync(0xffffffffu, t0 <= 32u && t1 <= 32u);
      if (use) {
#pragma unroll
        for (int j = 0; j < 3; ++j) {
          sts32_if(((t0 + j) & 3u) != 0u, row0 + (t0 + j) * 4, kPadKey);
          sts32_if(((t1 + j) & 3u) != 0u, row1 + (t1 + j) * 4, kPadKey);
          sts32_if(((t0 + j) & 3u) != 0u, row0 + kPbPosDelta + (t0 + j) * 4, 0xFFFFFFFFu);
          sts32_if(((t1 + j) & 3u) != 0u, row1 + kPbPosDelta + (t1 + j) * 4, 0xFFFFFFFFu);
        }
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
    if (!use) {  // the network kernel takes this array after this grid
      if (lane == 0) fail[1 + atomicAdd(&fail[0], 1u)] = (uint32_t)a;
      __syncwarp();
      continue;
    }
    uint32_t p[32];
#pragma unroll 1
    for (int rho = 0; rho < 2; ++rho) {
      const uint32_t tb = rho ? t0 : t1;
      const uint32_t row = rho ? row0 : row1;
      const uint32_t ob = (rho ? base0 : base1) * 4;
      if (rho == 0) {
#pragma unroll
        for (int i = 0; i < 32; ++i) { k[i] = kPadKey; p[i] = 0xFFFFFFFFu; }
      }
#pragma unroll
      for (int q = 0; q < 8; ++q) {
        lds128_if(4u * q < tb, row + q * 16, k[4 * q], k[4 * q + 1], k[4 * q + 2], k[4 * q + 3]);
        lds128_if(4u * q < tb, row + kPbPosDelta + q * 16, p[4 * q], p[4 * q + 1], p[4 * q + 2], p[4 * q + 3]);
      }
      __syncwarp();  // rows 32..63 are drained before any output is staged over them
      sort32_kp(k, p);
#pragma unroll
      for (int i = 0; i < 32; ++i) {
        sts32_if((uint32_t)i < tb, kst_sa + ob + i * 4, k[i]);
        sts32_if((uint32_t)i < tb, pst_sa + ob + i * 4, p[i]);
      }
    }
    __syncwarp();
    // payloads by position (L1: the row was touched by nobody else), all before the first store
    const uint32_t* vsrc = vals + a * (int64_t)n;
#pragma unroll
    for (int q = 0; q < 8; ++q) {
      const int c = lane + 32 * q;
      if (q < 4 || c < nc) {
        const uint4 pos = lds128(pst_sa + c * 16);
        p[4 * q] = vsrc[pos.x]; p[4 * q + 1] = vsrc[pos.y]; p[4 * q + 2] = vsrc[pos.z]; p[4 * q + 3] = vsrc[pos.w];
      }
    }
    __syncwarp();
#pragma unroll
    for (int q = 0; q < 8; ++q) {
      const int c = lane + 32 * q;
      uint4 kv = lds128(kst_sa + c * 16);
      if (!raw) { kv.x = bits_from_key(kv.x); kv.y = bits_from_key(kv.y); kv.z = bits_from_key(kv.z); kv.w = bits_from_key(kv.w); }
      stg_cs_if(q < 4 || c < nc, kdst + c, kv);
      stg_cs_if(q < 4 || c < nc, vdst + c, make_uint4(p[4 * q], p[4 * q + 1], p[4 * q + 2], p[4 * q + 3]));
    }
    __syncwarp();
  }
}

}  // namespace gas
