// Mandelbrot customizing function over PAIRS of neighbouring pixels, with
// Blackwell's packed two-lane FP32 instructions (eq. (5),
// P:L379-397; reading R4).  The element is a pair of positions {c0, c1} (a
// Vector<Pos2> has exactly the bytes of a Vector<Pos> of twice the length, so
// the image and the counts keep their row-major layout); the result is the
// pair of counts.
//
// Every update of every pixel is computed by exactly the operations of
// mandelbrot.cu, in the same order, each rounded once (FMA contraction off):
//   S = x*x + y*y (escape test),  xt = (x*x - y*y) + c.re,  y = (2x)*y + c.im.
// Two pixels share each instruction: FADD2 / FFMA2 on a register pair.  A
// multiply is written as fma(a, b, -0.0) with the -0.0 read from memory at run
// time: a*b + (-0.0) rounds exactly like a*b (for every a, b, including signed
// zeros, infinities and NaN), and ptxas cannot fuse it with the add that uses
// it (it does fuse mul.rn.f32x2 + add.rn.f32x2 into FFMA2, even with
// --fmad=false).  So the counts are bit-identical to eq. (5) as written --
// tested against the oracle and the golden CRCs.
//
// Structure per pair: (1) each pixel runs the plain loop for up to MANDEL_P
// updates (most non-members escape there: 93.5% within 8 on the paper image);
// (2) while both are alive, blocks of MANDEL_PB packed updates with the escape
// test of every update OR-ed into one flag per pixel; a block in which either
// escaped is rolled back to its start; (3) each pixel finishes alone with the
// blocked scalar loop (mandelbrot_blocked.cu's scheme).  Members (the bulk of
// the work) spend 5 instructions per update instead of 9.
#ifndef MANDEL_P
#define MANDEL_P 8
#endif
#ifndef MANDEL_PB
#define MANDEL_PB 8
#endif
#ifndef MANDEL_B
#define MANDEL_B 8
#endif
struct Pos2 { float re0, im0, re1, im1; };
struct Cnt2 { int n0, n1; };

#ifdef __CUDA_ARCH__
typedef unsigned long long mandel_f2;  // two floats in one 64-bit register pair (lo = pixel 0)
// -0.0 in both halves, read at run time so the multiplies stay unfused
__device__ mandel_f2 mandel_negzero2 = 0x8000000080000000ull;
static __forceinline__ mandel_f2 mk2(float lo, float hi) {
    return ((mandel_f2)__float_as_uint(hi) << 32) | (mandel_f2)__float_as_uint(lo);
}
static __forceinline__ float lo2(mandel_f2 v) { return __uint_as_float((unsigned)v); }
static __forceinline__ float hi2(mandel_f2 v) { return __uint_as_float((unsigned)(v >> 32)); }
static __forceinline__ mandel_f2 mul2z(mandel_f2 a, mandel_f2 b, mandel_f2 nz) {
    mandel_f2 d;
    asm("fma.rn.f32x2 %0, %1, %2, %3;" : "=l"(d) : "l"(a), "l"(b), "l"(nz));
    return d;
}
static __forceinline__ mandel_f2 add2(mandel_f2 a, mandel_f2 b) {
    mandel_f2 d;
    asm("add.rn.f32x2 %0, %1, %2;" : "=l"(d) : "l"(a), "l"(b));
    return d;
}
static __forceinline__ mandel_f2 sub2(mandel_f2 a, mandel_f2 b) {
    mandel_f2 d;
    asm("sub.rn.f32x2 %0, %1, %2;" : "=l"(d) : "l"(a), "l"(b));
    return d;
}
static __forceinline__ mandel_f2 load_negzero2() { return *(volatile mandel_f2 *)&mandel_negzero2; }
static __forceinline__ bool same2(mandel_f2 a, mandel_f2 b) { return a == b; }  // bit for bit
#else
// host build of this function (tests/test_workload_functions_host.py): the same
// arithmetic one float at a time (compiled with -ffp-contract=off)
struct mandel_f2 { float lo, hi; };
static inline mandel_f2 mk2(float lo, float hi) { return mandel_f2{lo, hi}; }
static inline float lo2(mandel_f2 v) { return v.lo; }
static inline float hi2(mandel_f2 v) { return v.hi; }
static inline mandel_f2 mul2z(mandel_f2 a, mandel_f2 b, mandel_f2 nz) {
    return mandel_f2{a.lo * b.lo + nz.lo, a.hi * b.hi + nz.hi};
}
static inline mandel_f2 add2(mandel_f2 a, mandel_f2 b) { return mandel_f2{a.lo + b.lo, a.hi + b.hi}; }
static inline mandel_f2 sub2(mandel_f2 a, mandel_f2 b) { return mandel_f2{a.lo - b.lo, a.hi - b.hi}; }
static inline mandel_f2 load_negzero2() { return mandel_f2{-0.0f, -0.0f}; }
#include <cstring>
static inline bool same2(mandel_f2 a, mandel_f2 b) { return std::memcmp(&a, &b, sizeof a) == 0; }
#endif
// MANDEL_PERIODIC: exact periodicity checking for the pair (as in
// mandelbrot_blocked.cu): after each packed block both pixels' states are
// compared bit for bit with the states saved at block 1, 2, 4, ... (Brent's
// schedule); if BOTH repeat, neither ever escapes and both counts are the cap
#ifndef MANDEL_PERIODIC
#define MANDEL_PERIODIC 0
#endif

// plain loop (eq. (5) as written) for at most `lim` updates from (x, y, n)
static __forceinline__ int mandel_plain(float cr, float ci, float &x, float &y, int n, int lim) {
    while (n < lim && x * x + y * y <= 4.0f) {
        float xt = (x * x - y * y) + cr;
        y = (2.0f * x) * y + ci;
        x = xt;
        ++n;
    }
    return n;
}

// blocked scalar loop (mandelbrot_blocked.cu) from (x, y, n) to the cap
template <int B> static __forceinline__ int mandel_finish(float cr, float ci, float x, float y, int n, int cap) {
    while (n + B <= cap) {
        const float x0 = x, y0 = y;
        bool out = false;
#pragma unroll
        for (int k = 0; k < B; ++k) {
            const float xx = x * x, yy = y * y;
            out = out | !(xx + yy <= 4.0f);
            const float xt = (xx - yy) + cr;
            y = (2.0f * x) * y + ci;
            x = xt;
        }
        if (out) {
            x = x0;
            y = y0;
            break;
        }
        n += B;
    }
    return mandel_plain(cr, ci, x, y, n, cap);
}

Cnt2 mandelbrot_pairs(Pos2 c, int cap) {
    float x0 = 0.0f, y0 = 0.0f, x1 = 0.0f, y1 = 0.0f;
    const int p = cap < MANDEL_P ? cap : MANDEL_P;
    int n0 = mandel_plain(c.re0, c.im0, x0, y0, 0, p);
    int n1 = mandel_plain(c.re1, c.im1, x1, y1, 0, p);
    if (n0 == p && n1 == p) {  // both alive: packed blocks
        const mandel_f2 nz = load_negzero2();
        const mandel_f2 cr = mk2(c.re0, c.re1), ci = mk2(c.im0, c.im1);
        mandel_f2 X = mk2(x0, x1), Y = mk2(y0, y1);
        int n = p;
#if MANDEL_PERIODIC
        mandel_f2 SX = X, SY = Y;
        int blk = 0, next_save = 1;
#endif
        while (n + MANDEL_PB <= cap) {
            const mandel_f2 Xs = X, Ys = Y;
            bool out0 = false, out1 = false;
#pragma unroll
            for (int k = 0; k < MANDEL_PB; ++k) {
                const mandel_f2 XX = mul2z(X, X, nz), YY = mul2z(Y, Y, nz);
                const mandel_f2 S = add2(XX, YY);
                out0 = out0 | !(lo2(S) <= 4.0f);
                out1 = out1 | !(hi2(S) <= 4.0f);
                const mandel_f2 XT = add2(sub2(XX, YY), cr);
                Y = add2(mul2z(add2(X, X), Y, nz), ci);
                X = XT;
            }
            if (out0 | out1) {  // one escaped inside this block: roll back, finish alone
                X = Xs;
                Y = Ys;
                break;
            }
            n += MANDEL_PB;
#if MANDEL_PERIODIC
            if (same2(X, SX) && same2(Y, SY)) {  // both orbits repeat exactly: members
                Cnt2 m;
                m.n0 = cap;
                m.n1 = cap;
                return m;
            }
            if (++blk == next_save) {
                SX = X;
                SY = Y;
                next_save <<= 1;
            }
#endif
        }
        x0 = lo2(X);
        y0 = lo2(Y);
        x1 = hi2(X);
        y1 = hi2(Y);
        n0 = n;
        n1 = n;
    }
    Cnt2 r;
    r.n0 = (n0 < p) ? n0 : mandel_finish<MANDEL_B>(c.re0, c.im0, x0, y0, n0, cap);
    r.n1 = (n1 < p) ? n1 : mandel_finish<MANDEL_B>(c.re1, c.im1, x1, y1, n1, cap);
    return r;
}
