// Mandelbrot customizing function, blocked form: the
// same iteration as mandelbrot.cu (eq. (5); reading R4) with the
// loop control paid once per block of MANDEL_B updates instead of per update.
// Inside a block every update still evaluates the paper's escape test
// x*x + y*y <= 4 on the current z, but only ORs it into a flag; a block in
// which z escaped is rolled back to its start and replayed one update at a
// time by the plain loop.  Every update that counts is therefore computed by
// exactly the operations of mandelbrot.cu in the same order (FMA contraction
// off), so the counts are bit-identical -- tested against the oracle and the
// golden image CRCs.  What changes is the instruction mix: per update 8 FP32
// operations + 1 compare instead of + 1 compare, 1 counter add, 1 counter
// compare and 1 branch.
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
#if MANDEL_PERIODIC
#ifndef __CUDA_ARCH__
#include <cstring>
static inline unsigned mandel_bits(float f) { unsigned u; std::memcpy(&u, &f, 4); return u; }
#else
static __forceinline__ unsigned mandel_bits(float f) { return __float_as_uint(f); }
#endif
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
#if MANDEL_PERIODIC
    unsigned sx = mandel_bits(x), sy = mandel_bits(y);  // saved state (block 0)
    int blk = 0, next_save = 1;
#endif
    while (n + B <= cap) {
        const float x0 = x, y0 = y;
        bool out = false;
#pragma unroll
        for (int k = 0; k < B; ++k) {
            const float xx = x * x, yy = y * y;
            out = out | !(xx + yy <= 4.0f);
            const float xt = (xx - yy) + c.re;
            y = (2.0f * x) * y + c.im;
            x = xt;
        }
        if (out) {  // escaped inside this block: replay it update by update
            x = x0;
            y = y0;
            break;
        }
        n += B;
#if MANDEL_PERIODIC
        if (mandel_bits(x) == sx && mandel_bits(y) == sy) return cap;  // exact cycle: a member
        if (++blk == next_save) {
            sx = mandel_bits(x);
            sy = mandel_bits(y);
            next_save <<= 1;
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
