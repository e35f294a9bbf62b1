/*
 * gas_oracle.c — CPU ORACLE for the GPU-ArraySort hot path.
 *
 * TEST INFRASTRUCTURE ONLY. Only tests/, __graft_entry__.smoke() and
 * bench.py's cpu_baseline / --impl reference legs may load this library.
 * It shares no code, header, table or constant with the CUDA path
 * (paper_conf_icppw_awans16_b200/csrc/); the two meet only at the seeded
 * input generators in datagen/.
 *
 * What it computes (PAPER.md, "P:L" = line of /root/reference/PAPER.md):
 *   Definition 1 (§4): for every array A_i of the batch I, output
 *   A'_i = the elements of A_i arranged so that a1 <= a2 <= ... <= an.
 *   Arrays are independent; the result overwrites the
 *   input in place (Abstract P:L38-39); elements are float32
 *   (§7.2).
 *
 * Reading C-1: "<=" on float32 is IEEE 754-2008
 * §5.10 totalOrder, so that -0, +0 and NaNs have a unique place and the
 * output is a permutation of the input BIT PATTERNS. Data is moved only as
 * uint32 bit patterns; floats are used only inside the comparison.
 *
 * The oracle is the plain definition: per array, C library qsort() with a
 * comparator that is §5.10 written out case by case (not a bit trick).
 * Single-threaded per call; callers may run disjoint array ranges on
 * several threads (no shared state).
 *
 * Build: gcc -O2 -fno-fast-math -std=c11 -shared -fPIC -o liboracle.so gas_oracle.c
 */
#include <math.h>
#include <stdint.h>
#include <stdlib.h>
#include <string.h>

#if defined(__FAST_MATH__)
#error "the oracle must be compiled without -ffast-math (IEEE comparisons)"
#endif

static float as_float(uint32_t b) { float f; memcpy(&f, &b, sizeof f); return f; }

/*
 * totalOrder(x, y) of IEEE 754-2008 §5.10 for binary32, returning 1 iff
 * x precedes or equals y:
 *   a) if x < y numerically, true; if x > y, false;
 *   b) if x == y numerically: -0 precedes +0 (totalOrder(-0,+0) true,
 *      totalOrder(+0,-0) false); otherwise equal representations -> true;
 *   c) if x or y is NaN: a negative-signed NaN precedes every number and
 *      every positive-signed NaN follows every number; two NaNs of the same
 *      sign are ordered, for positive sign, signaling before quiet and then
 *      by payload ascending — the reverse for negative sign.
 * The quiet bit of binary32 is the leading trailing-significand bit (bit 22),
 * so "(quiet, payload) ascending" is the 23-bit trailing field ascending.
 */
static int total_order(uint32_t xb, uint32_t yb)
{
    const float x = as_float(xb), y = as_float(yb);
    const int xneg = (int)(xb >> 31), yneg = (int)(yb >> 31);
    const int xnan = isnan(x), ynan = isnan(y);

    if (xnan || ynan) {                       /* case c) */
        if (xnan && ynan) {
            if (xneg != yneg) return xneg;    /* -NaN before +NaN */
            const uint32_t xt = xb & 0x007FFFFFu, yt = yb & 0x007FFFFFu;
            return xneg ? (xt >= yt) : (xt <= yt);
        }
        if (xnan) return xneg;                /* -NaN <= anything; +NaN <= only +NaNs (handled above) */
        return !yneg;                         /* x <= +NaN; x <= -NaN is false */
    }
    if (x < y) return 1;                      /* case a) */
    if (x > y) return 0;
    if (x == 0.0f) return xneg >= yneg;       /* case b): -0 before +0 */
    return 1;                                 /* same value, same representation */
}

static int cmp_total(const void* pa, const void* pb)
{
    const uint32_t a = *(const uint32_t*)pa, b = *(const uint32_t*)pb;
    const int ab = total_order(a, b), ba = total_order(b, a);
    if (ab && ba) return 0;
    return ab ? -1 : 1;
}

/* Exposed for the tests: totalOrder as a predicate on bit patterns. */
int gas_oracle_total_order(uint32_t xb, uint32_t yb) { return total_order(xb, yb); }

/*
 * Definition 1 on the fixed-length batch: N arrays of n
 * float32 each, array i at h[i*n .. i*n+n), each sorted ascending in place.
 * N <= 0 or n <= 1 is a no-op (reading C-4).
 */
void gas_oracle_sort_arrays(uint32_t* h, int64_t N, int32_t n)
{
    if (N <= 0 || n <= 1) return;
    for (int64_t i = 0; i < N; ++i)
        qsort(h + i * (int64_t)n, (size_t)n, sizeof(uint32_t), cmp_total);
}

/*
 * Variable-length variant (BASELINE.json north_star; reading C-16): array i
 * is h[off[i] .. off[i+1]), CSR offsets int64[N+1], nondecreasing.
 */
void gas_oracle_sort_arrays_offsets(uint32_t* h, const int64_t* off, int64_t N)
{
    for (int64_t i = 0; i < N; ++i) {
        const int64_t len = off[i + 1] - off[i];
        if (len > 1) qsort(h + off[i], (size_t)len, sizeof(uint32_t), cmp_total);
    }
}

/*
 * Key + payload variant (north_star "optional key+payload variant";
 * reading C-2): stable — elements with equal keys keep their input order,
 * so the payload order is unique. Stability is obtained the plain way:
 * ties in totalOrder are broken by the original position.
 */
typedef struct { uint32_t key, val; int64_t pos; } rec_t;

static int cmp_rec(const void* pa, const void* pb)
{
    const rec_t* a = (const rec_t*)pa;
    const rec_t* b = (const rec_t*)pb;
    const int c = cmp_total(&a->key, &b->key);
    if (c) return c;
    return (a->pos > b->pos) - (a->pos < b->pos);
}

int gas_oracle_sort_pairs(uint32_t* keys, uint32_t* vals, int64_t N, int32_t n)
{
    if (N <= 0 || n <= 1) return 0;
    rec_t* r = (rec_t*)malloc(sizeof(rec_t) * (size_t)n);
    if (!r) return -1;
    for (int64_t i = 0; i < N; ++i) {
        uint32_t* k = keys + i * (int64_t)n;
        uint32_t* v = vals + i * (int64_t)n;
        for (int32_t j = 0; j < n; ++j) { r[j].key = k[j]; r[j].val = v[j]; r[j].pos = j; }
        qsort(r, (size_t)n, sizeof(rec_t), cmp_rec);
        for (int32_t j = 0; j < n; ++j) { k[j] = r[j].key; v[j] = r[j].val; }
    }
    free(r);
    return 0;
}
