// split1024.cuh — value buckets for the arrays the plain bucket kernel
// (bucket1024.cuh) cannot take: IEEE special values (±NaN, ±inf, ±0,
// subnormals, the ±0 / NaN mix of BASELINE.json configs[4]) and
// duplicate-heavy arrays (a value repeated more often than a bucket holds).
// One warp per array, 512 < n <= 1024; kernel k_s1_split of the sort1024
// pipeline (sort1024.cuh).
//
// The paper's data-independent buckets (§4.1) need a value range;
// NaN and infinities have none, and equal values cannot be split by any map.
// Both are handled without a whole-array fallback:
//  * special values are classified per key (exponent 0 / 255, mantissa 0,
//    sign, quiet bit) and either counted (-inf, -0, +0, +inf: runs of one
//    known key, written as runs) or given their own bucket row (-qNaN, -sNaN,
//    negative subnormals, positive subnormals, +sNaN, +qNaN: sorted by the
//    row network like any bucket). Only the normal values go through the
//    value map, over [vlo, vhi] of the normal values alone;
//  * a bucket of more than 32 keys whose keys are all equal (every key that
//    did not fit in its 32 slots is folded into a per-row shared min / max) is
//    written as a run of that key.
// Rows in key order (IEEE 754 totalOrder, reading C-1), special
// arrays ("SP" path, b0 = value bucket of 0.0, normals in buckets 0..kSpTop):
//   0 -qNaN | 1 -sNaN | run -inf | 2 + b: negative normals (b <= b0) |
//   b0 + 3: negative subnormals | runs -0, +0 | b0 + 4: positive subnormals |
//   5 + b: positive normals (b >= b0) | run +inf | 62 +sNaN | 63 +qNaN.
// A negative normal value's bucket never exceeds b0 and a positive one's is
// never below it (the map is monotone), so the rows above are in order. Runs
// are attached to a neighbouring row in the bucket scan: -inf after row 1,
// the zeros after the negative subnormals, +inf before the keys of row 62.
// Arrays without NaN / inf (the "plain" path: duplicate-heavy data) use the
// 64 value buckets of bucket1024.cuh over [min, max] with the same equal-run
// overflow rule.
// Whatever is left — a row of more than 32 keys with two distinct keys, a
// value range that overflows — is re-read (L2) and sorted by the 1024-key
// network (warp1024.cuh). Correctness rests on the same monotone map as
// bucket1024.cuh and on the run rule checking equality of every key it folds.
#pragma once
#include <cstdint>

#include "bucket1024.cuh"
#include "sort1024.cuh"

namespace gas {

#ifndef GAS_SP_TMA  // 16-byte rows: stage float bits and leave through one TMA bulk store per array
#define GAS_SP_TMA 1   // measured: dup16 4.88 -> 4.61 ms, special_mix 6.98 -> 7.11 (only for plain arrays: special_mix 7.69)
#endif
#ifndef GAS_SP_BLOCK
#define GAS_SP_BLOCK 512  // measured (profiles/r02_ab_split_block.txt): 384 / 448 / 512 / 640 / 768 threads: dup16 4.94 / 4.81 / 4.53 / 4.57 / 4.85 ms, special_mix 7.83 / 7.59 / 6.61 / 6.74 / 7.14
#endif
constexpr int kSpBlock = GAS_SP_BLOCK;              // one block per SM
constexpr int kSpCntWords = 68;                     // 64 row counters + 4 run counters (-inf, -0, +0, +inf)
constexpr int kSpCntBytes = kSpCntWords * 4;
constexpr int kSpRowWords = 36;                     // 32 slots + words 32 / 33: min / max of the overflow keys
constexpr int kSpSlotBytes = 64 * kSpRowWords * 4;
constexpr int kSpStageWord = 32 * kSpRowWords;      // output word p at slot word kSpStageWord + p
constexpr int kSpWarpBytes = kSpCntBytes + kSpSlotBytes;
constexpr int kSpSmemBytes = (kSpBlock / 32) * kSpWarpBytes;
constexpr int kSpTop = 56;                          // SP path: normal values in value buckets 0..56 (rows 2..61)
static_assert(kSpSmemBytes <= 232448, "split kernel: shared memory per SM");
static_assert(5 + kSpTop <= 61, "split kernel: rows");

// Per-array map (warp-uniform). SP path: lo / s map the normal values,
// base_n / base_p turn the bucket bits (0x4B000000 + b) into rows 2 + b /
// 5 + b; tlo / thi_q / thi_s are the byte tables of the special rows.
struct SpMap {
  float lo, s;
  uint32_t base_n, base_p;
  uint32_t tlo, thi_q, thi_s;
};

// Row (0..63) or run counter (64..67) of one key (raw bits) on the SP path.
// Table index: bit 2 = exponent 255, bit 1 = mantissa 0, bit 0 = sign:
//   0 +subnormal, 1 -subnormal, 2 +0, 3 -0, 4 +NaN, 5 -NaN, 6 +inf, 7 -inf;
// NaN rows also depend on the quiet bit (thi_q / thi_s).
__device__ __forceinline__ uint32_t sp_row(uint32_t bits, const SpMap& m) {
  const uint32_t x = bits & 0x7F800000u;
  const bool normal = (x - 0x00800000u) < 0x7F000000u;
  const uint32_t rn = __float_as_uint(__fmaf_rn(__fsub_rn(__uint_as_float(bits), m.lo), m.s, 8388608.0f)) +
                      ((int32_t)bits < 0 ? m.base_n : m.base_p);
  const uint32_t idx = ((x >> 28) & 4u) | ((bits & 0x7FFFFFu) == 0u ? 2u : 0u) | (bits >> 31);
  const uint32_t rs = __byte_perm(m.tlo, (bits & 0x00400000u) ? m.thi_q : m.thi_s, idx) & 0xFFu;
  return normal ? rn : rs;
}

// Row of one key on the plain path (no NaN / inf): the 64 value buckets.
__device__ __forceinline__ uint32_t pl_row(uint32_t bits, float vmin, float s) {
  return bucket_bits(bits, vmin, s) - 0x4B000000u;
}

// Rank + scatter of one array's keys: the atomic returns the key's rank in
// its row; run keys (row >= 64) are only counted. A key of rank >= 32 does
// not fit: its row is written as a run if all its keys are equal. On the
// plain path (duplicate-heavy data: overflow is the rule) the key is compared
// here with the row's slot 0 (stored by the rank-0 key in this or an earlier
// group); the SP path, where overflow is rare, leaves it to
// sp_overflow_mismatch (no per-key cost when no row overflows). Returns
// whether one of this lane's keys differs.
template <bool SP, bool VEC>
__device__ __forceinline__ bool sp_scatter(const uint32_t (&k)[32], int lane, int n, const SpMap& m, float vmin,
                                           float s, uint32_t cnt_sa, uint32_t slot_sa) {
  bool mis = false;
#pragma unroll
  for (int g = 0; g < 32; g += 4) {
    uint32_t row[4], c[4];
#pragma unroll
    for (int r = g; r < g + 4; ++r) {
      row[r - g] = SP ? sp_row(k[r], m) : pl_row(k[r], vmin, s);
      c[r - g] = SP ? atoms_inc_if(cw_valid<VEC>(r, lane, n), cnt_sa + row[r - g] * 4)
                    : atoms_inc_pred(cw_valid<VEC>(r, lane, n), cnt_sa + row[r - g] * 4);
    }
    uint32_t ra[4], kk[4];
    bool ov[4];
#pragma unroll
    for (int r = g; r < g + 4; ++r) {
      const bool v = cw_valid<VEC>(r, lane, n) && (!SP || row[r - g] < 64u);
      kk[r - g] = key_from_bits(k[r]);
      ra[r - g] = slot_sa + row[r - g] * (kSpRowWords * 4);
      sts32_if(v && c[r - g] < 32u, ra[r - g] + c[r - g] * 4, kk[r - g]);
      ov[r - g] = v && c[r - g] >= 32u;
    }
    if (!SP && __any_sync(0xffffffffu, ov[0] || ov[1] || ov[2] || ov[3])) {
      __syncwarp();  // slot 0 of every row touched so far is stored
#pragma unroll
      for (int j = 0; j < 4; ++j) {
        uint32_t v = kk[j];  // slot 0 of the key's row when it overflowed, else the key itself
        asm volatile("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %1, 0;\n\t@q ld.shared.u32 %0, [%2];\n\t}"
                     : "+r"(v) : "r"((uint32_t)ov[j]), "r"(ra[j]) : "memory");
        mis |= v != kk[j];
      }
    }
  }
  return mis;
}

// SP path: every key of an overflowing row (masks om0: rows 0..31, om1: rows
// 32..63) must equal the row's slot 0. Returns whether one of this lane's
// keys does not.
template <bool VEC>
__device__ __forceinline__ bool sp_overflow_mismatch(const uint32_t (&k)[32], int lane, int n, const SpMap& m,
                                                     uint32_t slot_sa, uint32_t om0, uint32_t om1) {
  bool bad = false;
#pragma unroll
  for (int r = 0; r < 32; ++r) {
    const uint32_t row = sp_row(k[r], m);
    const uint32_t bit = ((row < 32u ? om0 : om1) >> (row & 31u)) & 1u;
    const bool over = cw_valid<VEC>(r, lane, n) && row < 64u && bit != 0u;
    const uint32_t kk = key_from_bits(k[r]);
    uint32_t v = kk;
    asm volatile("{\n\t.reg .pred q;\n\tsetp.ne.u32 q, %1, 0;\n\t@q ld.shared.u32 %0, [%2];\n\t}"
                 : "+r"(v) : "r"((uint32_t)over), "r"(slot_sa + row * (kSpRowWords * 4)) : "memory");
    bad |= v != kk;
  }
  return bad;
}

// Writes `len` copies of key `val` at staged positions [st, st + len) (one
// lane; 16-byte stores between the unaligned ends).
__device__ __forceinline__ void sp_fill(uint32_t stage_sa, uint32_t st, uint32_t len, uint32_t val) {
  uint32_t p = st;
  const uint32_t e = st + len;
  for (; p < e && (p & 3u); ++p) sts32(stage_sa + p * 4, val);
  for (; p + 4 <= e; p += 4) sts128(stage_sa + p * 4, make_uint4(val, val, val, val));
  for (; p < e; ++p) sts32(stage_sa + p * 4, val);
}

// The pipeline's split kernel: the whole batch when ctl->flag == kS1Split,
// else the arrays the counting-sort kernel listed. TB (16-byte rows): stage
// float bits and leave through one TMA bulk store per array — for batches the
// sampler found duplicate-heavy (dup16 4.88 -> 4.61 ms); batches it found
// special-heavy and the listed (special-heavy) arrays keep the key staging
// (special_mix 6.76 vs 6.95 ms with the bulk store).
template <bool VEC, bool TB>
__device__ __forceinline__ void split_body(uint32_t* __restrict__ d, int n, uint32_t one, const S1Ctl* ctl,
                                           uint32_t flag, int64_t count, uint4* sp_smem) {
  const uint32_t* list = s1_list(ctl);
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const uint32_t wsa = (uint32_t)__cvta_generic_to_shared(sp_smem) + warp * kSpWarpBytes;
  const uint32_t cnt_sa = wsa;
  const uint32_t slot_sa = wsa + kSpCntBytes;
  const uint32_t stage_sa = slot_sa + kSpStageWord * 4;
  uint32_t* const slot_ptr =
      reinterpret_cast<uint32_t*>(reinterpret_cast<unsigned char*>(sp_smem) + warp * kSpWarpBytes + kSpCntBytes);
  const uint32_t row0 = slot_sa + lane * (kSpRowWords * 4);  // this lane's rows: lane, lane + 32
  const uint32_t row1 = row0 + 32 * (kSpRowWords * 4);
  const int64_t nwarps = (int64_t)gridDim.x * (kSpBlock / 32);

  for (int64_t i = (int64_t)blockIdx.x * (kSpBlock / 32) + warp; i < count; i += nwarps) {
    const int64_t a = flag == kS1Split ? i : (int64_t)list[i];
    uint32_t* const arr = d + a * (int64_t)n;
    uint32_t k[32];
    s1_load<VEC>(k, arr, n, lane);
    if constexpr (TB) {
      bulk_wait_read_elect();  // the previous array's bulk store has read the staging rows
      __syncwarp();
    }
#if GAS_BK_PREFETCH
    prefetch_l2_elect(flag == kS1Split && i + nwarps < count, d + (i + nwarps) * (int64_t)n, n);
#endif
    // ---- key range: NaN / inf present? min / max of the normal values (SP) or of all keys (plain)
    uint32_t kmin = 0xFFFFFFFFu, kmax = 0u;
#pragma unroll
    for (int r = 0; r < 32; ++r) {
      const uint32_t kk = key_from_bits(k[r]);
      kmin = min(kmin, kk);
      kmax = max(kmax, kk);
    }
    kmin = __reduce_min_sync(0xffffffffu, kmin);
    kmax = __reduce_max_sync(0xffffffffu, kmax);
    const bool sp = !(kmin > 0x007FFFFFu && kmax < 0xFF800000u);  // a NaN or an infinity
    SpMap m;
    float vmin = 0.0f, s = 0.0f;
    bool ok = true;
    uint32_t zrow = 0;  // SP: the row the zero runs follow (negative subnormals)
    if (sp) {
      uint32_t nmin = 0xFFFFFFFFu, nmax = 0u;
#pragma unroll
      for (int r = 0; r < 32; ++r) {
        const uint32_t x = k[r] & 0x7F800000u;
        const bool normal = (x - 0x00800000u) < 0x7F000000u;
        const uint32_t kk = key_from_bits(k[r]);
        nmin = min(nmin, normal ? kk : 0xFFFFFFFFu);
        nmax = max(nmax, normal ? kk : 0u);
      }
      nmin = __reduce_min_sync(0xffffffffu, nmin);
      nmax = __reduce_max_sync(0xffffffffu, nmax);
      uint32_t b0 = 0;
      if (nmin <= nmax) {  // at least one normal value
        const float vlo = __uint_as_float(bits_from_key(nmin)), vhi = __uint_as_float(bits_from_key(nmax));
        const float range = __fsub_rn(vhi, vlo);
        s = range > 0.0f ? __fdiv_rn((float)kSpTop, range) : 0.0f;
        ok = range <= 3.402823466e38f && s <= 3.402823466e38f;
        vmin = vlo;
        if (vhi <= 0.0f) b0 = kSpTop;
        else if (vlo < 0.0f) b0 = pl_row(0u, vlo, s);  // 0 - vlo lies in (0, range): b0 in [0, kSpTop]
      }
      m.lo = vmin;
      m.s = s;
      m.base_n = 2u - 0x4B000000u;
      m.base_p = 5u - 0x4B000000u;
      zrow = b0 + 3u;
      m.tlo = (b0 + 4u) | ((b0 + 3u) << 8) | (66u << 16) | (65u << 24);
      m.thi_q = 63u | (0u << 8) | (67u << 16) | (64u << 24);
      m.thi_s = 62u | (1u << 8) | (67u << 16) | (64u << 24);
    } else {
      vmin = __uint_as_float(bits_from_key(kmin));
      const float range = __fsub_rn(__uint_as_float(bits_from_key(kmax)), vmin);
      s = range > 0.0f ? __fdiv_rn((float)GAS_BK_TOP, range) : 0.0f;
      ok = range <= 3.402823466e38f && s <= 3.402823466e38f;
    }

    bool bad = !ok;
    if (ok) {
      // ---- counters zero
      sts32(cnt_sa + lane * 4, 0u);
      sts32(cnt_sa + 128 + lane * 4, 0u);
      if (lane < 4) sts32(cnt_sa + 256 + lane * 4, 0u);
      __syncwarp();
      const bool mis = sp ? sp_scatter<true, VEC>(k, lane, n, m, vmin, s, cnt_sa, slot_sa)
                          : sp_scatter<false, VEC>(k, lane, n, m, vmin, s, cnt_sa, slot_sa);
      bad = __any_sync(0xffffffffu, mis);
      __syncwarp();
    }
    uint32_t t0 = 0, t1 = 0, base0 = 0, base1 = 0, r_ninf = 0, r_nz = 0, r_pz = 0, r_pinf = 0;
    if (ok) {
      t0 = lds32(cnt_sa + lane * 4);
      t1 = lds32(cnt_sa + 128 + lane * 4);
      if (sp) {
        const uint32_t om0 = __ballot_sync(0xffffffffu, t0 > 32u), om1 = __ballot_sync(0xffffffffu, t1 > 32u);
        if (om0 | om1) bad = __any_sync(0xffffffffu, sp_overflow_mismatch<VEC>(k, lane, n, m, slot_sa, om0, om1));
      }
      if (sp) {
        r_ninf = lds32(cnt_sa + 256);
        r_nz = lds32(cnt_sa + 260);
        r_pz = lds32(cnt_sa + 264);
        r_pinf = lds32(cnt_sa + 268);
      }
      // pads after the last key of each row, up to its 16-byte chunk boundary
#pragma unroll
      for (int j = 0; j < 3; ++j) {
        sts32_if(t0 < 32u && ((t0 + j) & 3u) != 0u, row0 + (t0 + j) * 4, kPadKey);
        sts32_if(t1 < 32u && ((t1 + j) & 3u) != 0u, row1 + (t1 + j) * 4, kPadKey);
      }
      // bucket bases: exclusive scan of the 64 row sizes plus the runs attached to them
      const uint32_t a0 = t0 + (lane == 1 ? r_ninf : 0u) + ((uint32_t)lane == zrow ? r_nz + r_pz : 0u);
      const uint32_t a1 = t1 + (lane == 30 ? r_pinf : 0u) + ((uint32_t)lane + 32u == zrow ? r_nz + r_pz : 0u);
      uint32_t x = a0 | (a1 << 16);
#pragma unroll
      for (int mm = 1; mm < 32; mm <<= 1) {
        const uint32_t y = __shfl_up_sync(0xffffffffu, x, mm);
        if (lane >= mm) x += y;
      }
      const uint32_t total_lo = __shfl_sync(0xffffffffu, x & 0xFFFFu, 31);
      base0 = (x & 0xFFFFu) - a0;
      base1 = total_lo + (x >> 16) - a1;
      __syncwarp();
    }

    // ---- two row rounds per lane: row lane + 32, then row lane
    uint32_t rep0 = 0, rep1 = 0;  // the key of an equal-key overflow row
    if (!bad) {
#pragma unroll 1
      for (int rho = 0; rho < 2; ++rho) {
        const uint32_t tb = rho ? t0 : t1;
        const uint32_t row = rho ? row0 : row1;
        const bool over = tb > 32u;
        // +inf run precedes the keys of row 62 (+sNaN)
        const uint32_t ob = stage_sa + ((rho ? base0 : base1) + (sp && rho == 0 && lane == 30 ? r_pinf : 0u)) * 4;
        if (rho == 0) {
#pragma unroll
          for (int q = 0; q < 32; ++q) k[q] = kPadKey;
        }
        const uint32_t tl = min(tb, 32u);
#pragma unroll
        for (int q = 0; q < 8; ++q) lds128_if(4u * q < tl, row + q * 16, k[4 * q], k[4 * q + 1], k[4 * q + 2], k[4 * q + 3]);
        const uint32_t rep = k[0];  // an overflowing row: all its keys must equal its slot 0
        if (__any_sync(0xffffffffu, over)) {
          uint32_t lo = k[0], hi = k[0];
#pragma unroll
          for (int q = 1; q < 31; q += 2) {
            lo = __vimin3_u32(lo, k[q], k[q + 1]);
            hi = __vimax3_u32(hi, k[q], k[q + 1]);
          }
          if (__any_sync(0xffffffffu, over && (lo != hi || k[31] != lo))) {
            bad = true;
            break;
          }
        }
        if (rho) rep0 = rep;
        else rep1 = rep;
        __syncwarp();  // rows 32..63 are drained before any output is staged over them
        const bool keys = !over && tb != 0u;
        if (__any_sync(0xffffffffu, keys)) {  // else every row of this round is empty or a run
          if (__any_sync(0xffffffffu, keys && tb >= 2u)) sortn_bk<32>(k, one);
          if (GAS_BK_MASKSTORE) {
            uint32_t* const sw = reinterpret_cast<uint32_t*>(sp_smem);
            stage_first<TB>(sw, (ob - (uint32_t)__cvta_generic_to_shared(sp_smem)) >> 2, keys ? tb : 0u, k);
          } else {
#pragma unroll
            for (int q = 0; q < 32; ++q) sts32_if(keys && (uint32_t)q < tb, ob + q * 4, TB ? bits_from_key(k[q]) : k[q]);
          }
        }
      }
    }
    if (!bad) {
      // ---- runs: equal-key overflow rows, then (SP) -inf, -0, +0, +inf
      // each lane writes its own overflow rows' runs; runs longer than 256 keys are written by the warp
      if (t1 > 32u && t1 <= 256u) sp_fill(stage_sa, base1, t1, TB ? bits_from_key(rep1) : rep1);
      if (t0 > 32u && t0 <= 256u) sp_fill(stage_sa, base0, t0, TB ? bits_from_key(rep0) : rep0);
      uint32_t om0 = __ballot_sync(0xffffffffu, t0 > 256u), om1 = __ballot_sync(0xffffffffu, t1 > 256u);
      while (om0 | om1) {
        const bool hi = om0 == 0u;
        const int owner = __ffs(hi ? om1 : om0) - 1;
        if (hi) om1 &= om1 - 1u;
        else om0 &= om0 - 1u;
        const uint32_t st = __shfl_sync(0xffffffffu, hi ? base1 : base0, owner);
        const uint32_t len = __shfl_sync(0xffffffffu, hi ? t1 : t0, owner);
        const uint32_t vk = __shfl_sync(0xffffffffu, hi ? rep1 : rep0, owner);
        const uint32_t val = TB ? bits_from_key(vk) : vk;
        for (uint32_t p = lane; p < len; p += 32) sts32(stage_sa + (st + p) * 4, val);
      }
      if (sp) {
        const uint32_t s_ninf = __shfl_sync(0xffffffffu, base0 + t0, 1);
        const uint32_t zs = __shfl_sync(0xffffffffu, zrow < 32u ? base0 + t0 : base1 + t1, (int)(zrow & 31u));
        const uint32_t s_pinf = __shfl_sync(0xffffffffu, base1, 30);
        // keys of -inf, -0, +0, +inf (TB: their bit patterns)
        for (uint32_t p = lane; p < r_ninf; p += 32) sts32(stage_sa + (s_ninf + p) * 4, TB ? 0xFF800000u : 0x007FFFFFu);
        for (uint32_t p = lane; p < r_nz; p += 32) sts32(stage_sa + (zs + p) * 4, TB ? 0x80000000u : 0x7FFFFFFFu);
        for (uint32_t p = lane; p < r_pz; p += 32) sts32(stage_sa + (zs + r_nz + p) * 4, TB ? 0x00000000u : 0x80000000u);
        for (uint32_t p = lane; p < r_pinf; p += 32) sts32(stage_sa + (s_pinf + p) * 4, TB ? 0x7F800000u : 0xFF800000u);
      }
      __syncwarp();
      // ---- store in place (keys -> bits)
      if constexpr (TB) {
        asm volatile("fence.proxy.async.shared::cta;" ::: "memory");  // staging writes -> async proxy
        __syncwarp();
        bulk_store_elect(arr, stage_sa, (uint32_t)n * 4u);
      } else if constexpr (VEC) {
        uint4* const dst = reinterpret_cast<uint4*>(arr);
        const int nc = n >> 2;
#pragma unroll
        for (int q = 0; q < 8; ++q) {
          const int c = lane + 32 * q;
          uint4 v = lds128(stage_sa + c * 16);
          v.x = bits_from_key(v.x); v.y = bits_from_key(v.y); v.z = bits_from_key(v.z); v.w = bits_from_key(v.w);
          stg_cs_if(q < 4 || c < nc, dst + c, v);
        }
      } else {
#pragma unroll
        for (int r = 0; r < 32; ++r) {
          const int e = lane + 32 * r;
          if (r < 16 || e < n) st_stream(arr + e, bits_from_key(lds32(stage_sa + e * 4)));
        }
      }
    } else {
      // ---- the array is untouched in memory: re-read it and sort it with the network
      __syncwarp();
      s1_load<VEC>(k, arr, n, lane);
      if constexpr (VEC) bucket1024_fallback(k, reinterpret_cast<uint4*>(arr), n >> 2, lane, slot_ptr, one);
      else bucket1024_fallback_scalar(k, arr, n, lane, slot_ptr, one);
    }
    __syncwarp();
  }
  if (TB) asm volatile("{\n\t.reg .pred e;\n\telect.sync _|e, 0xffffffff;\n\t@e cp.async.bulk.wait_group 0;\n\t}" ::: "memory");  // bulk stores complete before exit
}

template <bool VEC>
__global__ void __launch_bounds__(kSpBlock, 1) k_s1_split(uint32_t* __restrict__ d, int64_t N, int n, uint32_t one,
                                                          S1Ctl* ctl) {
  extern __shared__ __align__(16) uint4 sp_smem[];
  const uint32_t flag = ctl->flag;
  const int64_t count = flag == kS1Split ? N : (int64_t)ctl->nlist;
  if (count == 0) return;
  if (VEC && GAS_SP_TMA && flag == kS1Split && ctl->split_kind == kSplitDup)
    split_body<VEC, VEC && GAS_SP_TMA>(d, n, one, ctl, flag, count, sp_smem);
  else
    split_body<VEC, false>(d, n, one, ctl, flag, count, sp_smem);
}

}  // namespace gas
