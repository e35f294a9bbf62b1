// bitonic.cuh — in-register / warp-shuffle / shared-memory bitonic sorting
// network for one array of P = KPT * G * W ordered keys.
//
// Role in the method: this is step a5 of SURVEY.md §8(a) ("segment sort"),
// the replacement for the paper's Phase 1-3 sample sort (Alg. 1-3,
// P:L210-321). It keeps the paper's decomposition — each array is owned by
// one execution unit and arrays never interact — and its design
// rules (no divergent branches, shared memory for on-chip exchange,
// P:L154-167), but sorts with a data-oblivious network so that time does not
// depend on the value distribution (duplicates, pre-sorted input).
//
// Layout: element index i (0..P-1) of the array lives in
//     register r = i % KPT  of  lane g = (i / KPT) % G  of  warp w = i / (KPT*G)
// within the group of G lanes (G <= 32, aligned inside the warp) and W warps
// that own the array. Stages on register bits are compare-exchanges inside a
// thread (compile-time min/max), stages on lane bits use SHFL.BFLY, stages on
// warp bits go through shared memory.
//
// Network: the "mirror" formulation of bitonic sort — merge step of size K
// first compares i with i ^ (K-1), then half-cleaners at distances
// K/4 ... 1 — so every compare-exchange is ascending (lower index gets the
// minimum) and no per-block direction bit is needed.
#pragma once
#include <cstdint>

namespace gas {

// Barrier of a thread group: bar == 0 -> the whole CTA (__syncthreads);
// else named barrier (bar & 0xFF) over (bar >> 8) threads (several arrays
// sorted by independent thread groups of one CTA, bucket_cta.cuh).
__device__ __forceinline__ void group_sync(uint32_t bar) {
  if (bar == 0) __syncthreads();
  else asm volatile("bar.sync %0, %1;" ::"r"(bar & 0xFFu), "r"(bar >> 8) : "memory");
}
__device__ __forceinline__ bool group_and(bool v, uint32_t bar) {
  if (bar == 0) return __syncthreads_and(v);
  uint32_t r;
  asm volatile("{\n\t.reg .pred p, q;\n\tsetp.ne.u32 p, %1, 0;\n\tbar.red.and.pred q, %2, %3, p;\n\tselp.u32 %0, 1, 0, q;\n\t}"
               : "=r"(r) : "r"((uint32_t)v), "r"(bar & 0xFFu), "r"(bar >> 8) : "memory");
  return r != 0;
}

template <int X>
struct Log2 { static constexpr int value = 1 + Log2<X / 2>::value; };
template <>
struct Log2<1> { static constexpr int value = 0; };

// Compare-exchange, ascending. The min always runs on the integer ALU pipe;
// the max is either a second VIMNMX (ALU pipe) or (a + b) - min computed with
// two IMADs on the FMA pipe (exact in mod-2^32 arithmetic). `one` is an
// opaque register holding 1 so that ptxas keeps the IMAD form. Mixing the two
// forms balances the ALU and FMA pipes (tools/microbench.cu: both 64 op/clk/SM).
template <bool FMA>
__device__ __forceinline__ void ce(uint32_t& a, uint32_t& b, uint32_t one) {
  const uint32_t mn = min(a, b);
  if constexpr (FMA) {
    uint32_t s, mx;
    asm("mad.lo.u32 %0, %1, %2, %3;" : "=r"(s) : "r"(a), "r"(one), "r"(b));
    asm("mad.lo.u32 %0, %1, %2, %3;" : "=r"(mx) : "r"(mn), "r"(0u - one), "r"(s));
    b = mx;
  } else {
    b = max(a, b);
  }
  a = mn;
}

// Which compare-exchanges take the FMA form: MIX_NUM out of every MIX_DEN.
#ifndef GAS_CE_MIX_NUM
#define GAS_CE_MIX_NUM 2
#endif
#ifndef GAS_CE_MIX_DEN
#define GAS_CE_MIX_DEN 3
#endif

__device__ __forceinline__ void ce_n(int c, uint32_t& a, uint32_t& b, uint32_t one) {
  // c is a compile-time constant after unrolling, so the branch folds away.
  if ((c % GAS_CE_MIX_DEN) < GAS_CE_MIX_NUM) ce<true>(a, b, one);
  else ce<false>(a, b, one);
}

// 64-bit elements (key << 32 | original position: the stable pairs variant).
__device__ __forceinline__ void ce_n(int, uint64_t& a, uint64_t& b, uint32_t) {
  const uint64_t mn = a < b ? a : b;
  b = a < b ? b : a;
  a = mn;
}

// Keep the min (lower index) or the max (upper index) of x and the partner's y.
__device__ __forceinline__ uint32_t keep(uint32_t x, uint32_t y, bool upper) {
  return upper ? max(x, y) : min(x, y);
}
__device__ __forceinline__ uint64_t keep(uint64_t x, uint64_t y, bool upper) {
  return (upper == (x < y)) ? y : x;
}

template <int KPT, int G, int W, typename T = uint32_t>
struct Bitonic {
  static_assert(KPT >= 1 && (KPT & (KPT - 1)) == 0, "KPT power of two");
  static_assert(G >= 1 && G <= 32 && (G & (G - 1)) == 0, "G power of two <= 32");
  static_assert(W >= 1 && (W & (W - 1)) == 0 && (W == 1 || G == 32), "W>1 needs full warps");
  static constexpr int LOGK = Log2<KPT>::value;
  static constexpr int LOGG = Log2<G>::value;
  static constexpr int P = KPT * G * W;
  static constexpr int LOGP = Log2<P>::value;
  static constexpr int NT = 32 * W;  // threads per array when W > 1

  // In-register stage at distance j (< KPT): pairs (r, r|j) with bit j clear.
  template <int J>
  __device__ __forceinline__ static void reg_stage(T (&k)[KPT], uint32_t one) {
#pragma unroll
    for (int r = 0; r < KPT; ++r)
      if (!(r & J)) ce_n(r, k[r], k[r | J], one);
  }

  // In-register mirror stage of merge size K (<= KPT): pairs (r, r ^ (K-1)).
  template <int K>
  __device__ __forceinline__ static void reg_mirror(T (&k)[KPT], uint32_t one) {
#pragma unroll
    for (int r = 0; r < KPT; ++r)
      if (!(r & (K / 2))) ce_n(r, k[r], k[r ^ (K - 1)], one);
  }

  // Shared-memory exchange stage for partners in other warps. Element (t, r)
  // is stored at xs[r*T + t] (conflict-free for consecutive t).
  __device__ __forceinline__ static void smem_stage(T (&k)[KPT], T* xs, int t, int tmask,
                                                    int rmask, bool upper, uint32_t bar = 0) {
    group_sync(bar);
#pragma unroll
    for (int r = 0; r < KPT; ++r) xs[r * NT + t] = k[r];
    group_sync(bar);
    // tmask >= 32: the partner is in another warp and `upper` is a warp bit, so
    // this branch is warp-uniform and each key costs one min or one max
    if (upper) {
#pragma unroll
      for (int r = 0; r < KPT; ++r) k[r] = max(k[r], xs[(r ^ rmask) * NT + (t ^ tmask)]);
    } else {
#pragma unroll
      for (int r = 0; r < KPT; ++r) k[r] = min(k[r], xs[(r ^ rmask) * NT + (t ^ tmask)]);
    }
  }

  // Half-cleaner at distance 2^LJ, then the rest of the cascade down to 1.
  template <int LJ>
  __device__ __forceinline__ static void cleaners(T (&k)[KPT], int g, int t, T* xs, uint32_t one) {
    if constexpr (LJ >= 0) {
      constexpr int J = 1 << LJ;
      if constexpr (LJ < LOGK) {
        reg_stage<J>(k, one);
      } else if constexpr (LJ < LOGK + LOGG) {
        constexpr int m = J >> LOGK;
        const bool upper = g & m;
#pragma unroll
        for (int r = 0; r < KPT; ++r) k[r] = keep(k[r], __shfl_xor_sync(0xffffffffu, k[r], m), upper);
      } else {
        smem_stage(k, xs, t, J >> LOGK, 0, t & (J >> LOGK));
      }
      cleaners<LJ - 1>(k, g, t, xs, one);
    }
  }

  // Merge step of size K = 2^LK: mirror stage (partner i ^ (K-1)), then cleaners.
  template <int LK>
  __device__ __forceinline__ static void merge(T (&k)[KPT], int g, int t, T* xs, uint32_t one) {
    constexpr int K = 1 << LK;
    if constexpr (LK <= LOGK) {
      reg_mirror<K>(k, one);
    } else if constexpr (LK <= LOGK + LOGG) {
      constexpr int m = (K - 1) >> LOGK;
      const bool upper = g & ((K >> 1) >> LOGK);
      if constexpr (KPT == 1) {
        k[0] = keep(k[0], __shfl_xor_sync(0xffffffffu, k[0], m), upper);
      } else {
#pragma unroll
        for (int r = 0; r < KPT / 2; ++r) {
          const int r2 = KPT - 1 - r;
          const T v1 = __shfl_xor_sync(0xffffffffu, k[r2], m);
          const T v2 = __shfl_xor_sync(0xffffffffu, k[r], m);
          k[r] = keep(k[r], v1, upper);
          k[r2] = keep(k[r2], v2, upper);
        }
      }
    } else {
      smem_stage(k, xs, t, (K - 1) >> LOGK, KPT - 1, t & ((K >> 1) >> LOGK));
    }
    cleaners<LK - 2>(k, g, t, xs, one);
  }

  template <int LK>
  __device__ __forceinline__ static void sort_from(T (&k)[KPT], int g, int t, T* xs, uint32_t one) {
    if constexpr (LK <= LOGP) {
      merge<LK>(k, g, t, xs, one);
      sort_from<LK + 1>(k, g, t, xs, one);
    }
  }

  // Sort the P keys ascending. g: lane index inside the G-lane group;
  // t: thread index inside the array's W warps (t = w*32 + g; used when W > 1);
  // xs: P words of shared memory (used when W > 1).
  __device__ __forceinline__ static void sort(T (&k)[KPT], int g, int t, T* xs, uint32_t one) {
    sort_from<1>(k, g, t, xs, one);
  }
};

}  // namespace gas
