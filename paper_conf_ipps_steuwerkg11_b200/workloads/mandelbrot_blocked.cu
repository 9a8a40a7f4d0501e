// Mandelbrot customizing function, blocked form: the
// same iteration as mandelbrot.cu (eq. (5); reading R4) with the
// loop control paid once per block of MANDEL_B updates instead of per update.
// Inside a block every update still computes the paper's escape test value
// S = x*x + y*y, and the block's tests are decided together (MANDEL_MAXTEST,
// below: one NaN-propagating maximum; or each compare OR-ed into a flag); a
// block in which z escaped is rolled back to its start and replayed one update
// at a time by the plain loop.  Every update that counts is therefore computed
// by exactly the operations of mandelbrot.cu in the same order (FMA
// contraction off), so the counts are bit-identical -- tested against the
// oracle and the golden image CRCs.  What changes is the instruction mix: per
// update 8 FP32 operations + half a FMNMX3 instead of + 1 compare, 1 counter
// add, 1 counter compare and 1 branch.
// Block length: 8 updates, 16 for deep caps (a longer block pays off when
// most pixels run long; measured at 4096x3072: cap 256 best with 8, cap 4096
// with 16 -- 2.28 -> 2.04 ms).
#ifndef MANDEL_B
#define MANDEL_B 8
#endif
struct Pos { float re, im; };
// MANDEL_PRE: updates done by the plain loop before the blocks start -- most
// pixels outside the set escape within a few updates (93.5% within 8 on the
// paper image), and for them a first block would be computed, rolled back and
// replayed
#ifndef MANDEL_PRE
#define MANDEL_PRE 0
#endif
// MANDEL_PERIODIC: periodicity checking (exact).  After each block the state z
// is compared BIT FOR BIT with a z saved at an earlier block end (saved at
// block 1, 2, 4, 8, ... -- Brent's schedule, so any cycle length is caught).
// The iteration is a deterministic function of z (c is fixed), so equal states
// mean the orbit repeats forever; every test between the two block ends
// passed, so it never escapes and the count is the cap -- exactly what eq. (5)
// as written returns, without computing the rest (float32 orbits of interior
// points settle into exact cycles; 41% fewer updates on the paper's image).
#ifndef MANDEL_PERIODIC
#define MANDEL_PERIODIC 0
#endif
// block index of the next save of the periodicity check: doubling is Brent's
// schedule; any schedule whose gaps grow without bound finds every cycle (a
// detection is exact either way: equal states repeat forever)
#ifndef MANDEL_SAVE_NEXT
#define MANDEL_SAVE_NEXT(s) ((s) << 1)
#endif
#if MANDEL_PERIODIC
#ifndef __CUDA_ARCH__
#include <cstring>
static inline unsigned mandel_bits(float f) { unsigned u; std::memcpy(&u, &f, 4); return u; }
#else
static __forceinline__ unsigned mandel_bits(float f) { return __float_as_uint(f); }
#endif
#endif
// MANDEL_MAXTEST: the block's escape tests as ONE comparison.  Every update
// still computes the paper's S = x*x + y*y (rounded exactly as written), but
// instead of comparing each S with 4 the block keeps M = max(S_0, ..., S_{B-1})
// with a NaN-propagating maximum (PTX max.NaN.f32; ptxas folds two into one
// FMNMX3.NAN per two updates) and tests M <= 4 at the end: M <= 4 holds exactly when
// every S <= 4 holds (a NaN S makes M NaN and the block is rolled back, as a
// NaN S fails the paper's test).  Measured on the member loop: 87% of the
// FP32 lane peak against 73% for one compare per update (tools/fp32_probe.cu).
#ifndef MANDEL_MAXTEST
#define MANDEL_MAXTEST 1
#endif
// MANDEL_NOREPLAY: the maximum test of MANDEL_MAXTEST with the block's B test
// values kept, so an escape inside a block is resolved by finding the first
// failing test instead of rolling back and replaying (no divergent replay loop;
// with MANDEL_PRE 0 every pixel runs blocks only, the lanes of a warp in step).
#ifndef MANDEL_NOREPLAY
#define MANDEL_NOREPLAY 0
#endif
#ifdef __CUDA_ARCH__
static __forceinline__ float mandel_max2(float a, float b) {
    float d;
    asm("max.NaN.f32 %0, %1, %2;" : "=f"(d) : "f"(a), "f"(b));
    return d;
}
// two chained maxima: ptxas emits one FMNMX3.NAN
static __forceinline__ float mandel_max3(float a, float b, float c) { return mandel_max2(mandel_max2(a, b), c); }
#else
static inline float mandel_max2(float a, float b) { return (b > a || b != b) ? b : a; }  // NaN wins
static inline float mandel_max3(float a, float b, float c) { return mandel_max2(mandel_max2(a, b), c); }
#endif
template <int B> static int mandel_blocked(Pos c, int cap) {
    float x = 0.0f, y = 0.0f;
    int n = 0;
    if (MANDEL_PRE > 0) {
        const int p = cap < MANDEL_PRE ? cap : MANDEL_PRE;
        while (n < p && x * x + y * y <= 4.0f) {
            float xt = (x * x - y * y) + c.re;
            y = (2.0f * x) * y + c.im;
            x = xt;
            ++n;
        }
        if (n < p) return n;  // escaped in the prefix
    }
#if MANDEL_PERIODIC == 1
    unsigned sx = mandel_bits(x), sy = mandel_bits(y);  // saved state (block 0)
    int blk = 0, next_save = 1;
#endif
    while (n + B <= cap) {
#if MANDEL_NOREPLAY
        // every update of the block is computed; the B test values stay in
        // registers, so a block in which z escapes needs no replay: the count
        // ends at the first update whose test fails (updates after it are
        // discarded, whatever they computed -- inf or NaN included)
        float sv[B];
        float m = 0.0f;
#pragma unroll
        for (int k = 0; k < B; k += 2) {
            const float xx0 = x * x, yy0 = y * y;
            sv[k] = xx0 + yy0;
            const float xt0 = (xx0 - yy0) + c.re;
            y = (2.0f * x) * y + c.im;
            x = xt0;
            const float xx1 = x * x, yy1 = y * y;
            sv[k + 1] = xx1 + yy1;
            const float xt1 = (xx1 - yy1) + c.re;
            y = (2.0f * x) * y + c.im;
            x = xt1;
            m = mandel_max3(m, sv[k], sv[k + 1]);
        }
        if (!(m <= 4.0f)) {
            int k = B;
#pragma unroll
            for (int j = B - 1; j >= 0; --j)
                if (!(sv[j] <= 4.0f)) k = j;
            return n + k;
        }
#else
        const float x0 = x, y0 = y;
#if MANDEL_MAXTEST
        static_assert(B % 2 == 0, "MANDEL_MAXTEST folds the tests of two updates per FMNMX3");
        float m = 0.0f;
#pragma unroll
        for (int k = 0; k < B; k += 2) {
            const float xx0 = x * x, yy0 = y * y;
            const float s0 = xx0 + yy0;
            const float xt0 = (xx0 - yy0) + c.re;
            y = (2.0f * x) * y + c.im;
            x = xt0;
            const float xx1 = x * x, yy1 = y * y;
            const float s1 = xx1 + yy1;
            const float xt1 = (xx1 - yy1) + c.re;
            y = (2.0f * x) * y + c.im;
            x = xt1;
            m = mandel_max3(m, s0, s1);
        }
        const bool out = !(m <= 4.0f);
#else
        bool out = false;
#pragma unroll
        for (int k = 0; k < B; ++k) {
            const float xx = x * x, yy = y * y;
            out = out | !(xx + yy <= 4.0f);
            const float xt = (xx - yy) + c.re;
            y = (2.0f * x) * y + c.im;
            x = xt;
        }
#endif
        if (out) {  // escaped inside this block: replay it update by update
            x = x0;
            y = y0;
            break;
        }
#endif  // MANDEL_NOREPLAY
        n += B;
#if MANDEL_PERIODIC == 2
        // the state at the block's start (kept for the roll-back anyway): a
        // cycle whose length divides B (fixed points and the short cycles
        // float32 orbits of the large bulbs settle into) -- two compares per
        // block and no save schedule
        if (mandel_bits(x) == mandel_bits(x0) && mandel_bits(y) == mandel_bits(y0)) return cap;
#elif MANDEL_PERIODIC
        if (mandel_bits(x) == sx && mandel_bits(y) == sy) return cap;  // exact cycle: a member
        if (++blk == next_save) {
            sx = mandel_bits(x);
            sy = mandel_bits(y);
            next_save = MANDEL_SAVE_NEXT(next_save);
        }
#endif
    }
    while (n < cap && x * x + y * y <= 4.0f) {
        float xt = (x * x - y * y) + c.re;
        y = (2.0f * x) * y + c.im;
        x = xt;
        ++n;
    }
    return n;
}
int mandelbrot_blocked(Pos c, int cap) {
    return cap >= 1024 ? mandel_blocked<2 * MANDEL_B>(c, cap) : mandel_blocked<MANDEL_B>(c, cap);
}
