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
static __forceinline__ bool same_lo(mandel_f2 a, mandel_f2 b) { return (unsigned)a == (unsigned)b; }  // bit for bit
static __forceinline__ bool same_hi(mandel_f2 a, mandel_f2 b) { return (unsigned)(a >> 32) == (unsigned)(b >> 32); }
#else
#include <cstring>
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
static inline bool same_lo(mandel_f2 a, mandel_f2 b) { return std::memcmp(&a.lo, &b.lo, 4) == 0; }
static inline bool same_hi(mandel_f2 a, mandel_f2 b) { return std::memcmp(&a.hi, &b.hi, 4) == 0; }
#endif
// MANDEL_PERIODIC: exact periodicity checking for the pair (as in
// mandelbrot_blocked.cu): after each packed block both pixels' states are
// compared bit for bit with the states saved at block 1, 2, 4, ... (Brent's
// schedule); if BOTH repeat, neither ever escapes and both counts are the cap
#ifndef MANDEL_PERIODIC
#define MANDEL_PERIODIC 0
#endif
// block index of the next save of the periodicity check: doubling is Brent's
// schedule; any schedule whose gaps grow without bound finds every cycle (a
// detection is exact either way: equal states repeat forever)
#ifndef MANDEL_SAVE_NEXT
#define MANDEL_SAVE_NEXT(s) ((s) << 1)
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

// blocked scalar loop (mandelbrot_blocked.cu) from (x, y, n) to the cap, for
// the pixel of a pair that is still alive when the other escapes: with the
// block's tests folded into one maximum (MANDEL_MAXTEST, see
// mandelbrot_blocked.cu) and, with MANDEL_PERIODIC, exact periodicity checking
// (states compared bit for bit at block ends, saved at blocks 1, 2, 4, ...)
#ifndef MANDEL_MAXTEST
#define MANDEL_MAXTEST 1
#endif
#ifdef __CUDA_ARCH__
static __forceinline__ float mandel_max2(float a, float b) {
    float d;
    asm("max.NaN.f32 %0, %1, %2;" : "=f"(d) : "f"(a), "f"(b));
    return d;
}
// two chained maxima: ptxas emits one FMNMX3.NAN
static __forceinline__ float mandel_max3(float a, float b, float c) { return mandel_max2(mandel_max2(a, b), c); }
static __forceinline__ unsigned mandel_bits(float f) { return __float_as_uint(f); }
#else
static inline float mandel_max2(float a, float b) { return (b > a || b != b) ? b : a; }  // NaN wins
static inline float mandel_max3(float a, float b, float c) { return mandel_max2(mandel_max2(a, b), c); }
static inline unsigned mandel_bits(float f) { unsigned u; std::memcpy(&u, &f, 4); return u; }
#endif
template <int B> static __forceinline__ int mandel_finish(float cr, float ci, float x, float y, int n, int cap) {
#if MANDEL_PERIODIC
    unsigned sx = mandel_bits(x), sy = mandel_bits(y);
    int blk = 0, next_save = 1;
#endif
    while (n + B <= cap) {
        const float x0 = x, y0 = y;
#if MANDEL_MAXTEST
        float m = 0.0f;
#pragma unroll
        for (int k = 0; k < B; k += 2) {
            const float xx0 = x * x, yy0 = y * y;
            const float s0 = xx0 + yy0;
            const float xt0 = (xx0 - yy0) + cr;
            y = (2.0f * x) * y + ci;
            x = xt0;
            const float xx1 = x * x, yy1 = y * y;
            const float s1 = xx1 + yy1;
            const float xt1 = (xx1 - yy1) + cr;
            y = (2.0f * x) * y + ci;
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
            const float xt = (xx - yy) + cr;
            y = (2.0f * x) * y + ci;
            x = xt;
        }
#endif
        if (out) {
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
            next_save = MANDEL_SAVE_NEXT(next_save);
        }
#endif
    }
    return mandel_plain(cr, ci, x, y, n, cap);
}

// MANDEL_NOREPLAY: the pair stays in the packed loop until BOTH pixels are
// done, so the lanes of a warp never split into per-pixel finishing loops.  A
// block keeps its PB packed test values S (as in mandelbrot_blocked.cu's
// MANDEL_NOREPLAY): when a pixel escapes inside a block its count is the
// position of its first failing test, found without a replay, and from then on
// its half of each packed instruction computes values nobody reads (inf or
// NaN included).  A pixel whose orbit repeats bit for bit (MANDEL_PERIODIC) is
// done with the cap.  The tests of two updates are folded per pixel into one
// NaN-propagating maximum (FMNMX3), compared with 4 once per block.
#ifndef MANDEL_NOREPLAY
#define MANDEL_NOREPLAY 0
#endif
#ifndef MANDEL_NR_FSETP
#define MANDEL_NR_FSETP 0
#endif
#if MANDEL_NOREPLAY
static __forceinline__ Cnt2 mandel_pairs_nr(Pos2 c, int cap) {
    float x0 = 0.0f, y0 = 0.0f, x1 = 0.0f, y1 = 0.0f;
    const int p = cap < MANDEL_P ? cap : MANDEL_P;
    Cnt2 r;
    r.n0 = mandel_plain(c.re0, c.im0, x0, y0, 0, p);
    r.n1 = mandel_plain(c.re1, c.im1, x1, y1, 0, p);
    bool a0 = r.n0 == p, a1 = r.n1 == p;  // alive: no test has failed yet
    if (!(a0 || a1)) return r;
    const mandel_f2 nz = load_negzero2();
    const mandel_f2 cr = mk2(c.re0, c.re1), ci = mk2(c.im0, c.im1);
    mandel_f2 X = mk2(x0, x1), Y = mk2(y0, y1);
    int n = p;
#if MANDEL_PERIODIC
    mandel_f2 SX = X, SY = Y;
    int blk = 0, next_save = 1;
#endif
    while ((a0 || a1) && n + MANDEL_PB <= cap) {
        static_assert(MANDEL_PB % 2 == 0, "tests folded two updates at a time");
        mandel_f2 S[MANDEL_PB];
#if MANDEL_NR_FSETP
        // one compare per update and pixel, OR-ed into a flag (measured faster
        // than the folded maximum for the packed loop: tools/fp32_probe.cu)
        bool o0 = false, o1 = false;
#else
        float m0 = 0.0f, m1 = 0.0f;
#endif
#pragma unroll
        for (int k = 0; k < MANDEL_PB; ++k) {
            const mandel_f2 XX = mul2z(X, X, nz), YY = mul2z(Y, Y, nz);
            S[k] = add2(XX, YY);
            const mandel_f2 XT = add2(sub2(XX, YY), cr);
            Y = add2(mul2z(add2(X, X), Y, nz), ci);
            X = XT;
#if MANDEL_NR_FSETP
            o0 = o0 | !(lo2(S[k]) <= 4.0f);
            o1 = o1 | !(hi2(S[k]) <= 4.0f);
#else
            if (k & 1) {
                m0 = mandel_max3(m0, lo2(S[k - 1]), lo2(S[k]));
                m1 = mandel_max3(m1, hi2(S[k - 1]), hi2(S[k]));
            }
#endif
        }
#if MANDEL_NR_FSETP
        const bool e0 = o0, e1 = o1;
#else
        const bool e0 = !(m0 <= 4.0f), e1 = !(m1 <= 4.0f);
#endif
        if (a0 && e0) {  // pixel 0 escaped in this block: its first failing test
            int k = MANDEL_PB;
#pragma unroll
            for (int j = MANDEL_PB - 1; j >= 0; --j)
                if (!(lo2(S[j]) <= 4.0f)) k = j;
            r.n0 = n + k;
            a0 = false;
        }
        if (a1 && e1) {
            int k = MANDEL_PB;
#pragma unroll
            for (int j = MANDEL_PB - 1; j >= 0; --j)
                if (!(hi2(S[j]) <= 4.0f)) k = j;
            r.n1 = n + k;
            a1 = false;
        }
        n += MANDEL_PB;
#if MANDEL_PERIODIC
        if (a0 && same_lo(X, SX) && same_lo(Y, SY)) {  // exact cycle: a member
            r.n0 = cap;
            a0 = false;
        }
        if (a1 && same_hi(X, SX) && same_hi(Y, SY)) {
            r.n1 = cap;
            a1 = false;
        }
        if (++blk == next_save) {
            SX = X;
            SY = Y;
            next_save = MANDEL_SAVE_NEXT(next_save);
        }
#endif
    }
    // the last cap mod PB updates (none for cap 256), or the cap itself
    if (a0) {
        float x = lo2(X), y = lo2(Y);
        r.n0 = mandel_plain(c.re0, c.im0, x, y, n, cap);
    }
    if (a1) {
        float x = hi2(X), y = hi2(Y);
        r.n1 = mandel_plain(c.re1, c.im1, x, y, n, cap);
    }
    return r;
}
#endif

Cnt2 mandelbrot_pairs(Pos2 c, int cap) {
#if MANDEL_NOREPLAY
    return mandel_pairs_nr(c, cap);
#endif
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
        // per pixel: its orbit has repeated bit for bit (it never escapes; the
        // packed block keeps computing it until the other pixel is done too)
        bool done0 = false, done1 = false;
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
            // each pixel on its own: detecting only when BOTH states match their
            // saves at the same block end would wait for a common multiple of
            // the two cycle lengths
            done0 = done0 || (same_lo(X, SX) && same_lo(Y, SY));
            done1 = done1 || (same_hi(X, SX) && same_hi(Y, SY));
            if (done0 && done1) {  // both orbits repeat exactly: members
                Cnt2 m;
                m.n0 = cap;
                m.n1 = cap;
                return m;
            }
            if (++blk == next_save) {
                SX = X;
                SY = Y;
                next_save = MANDEL_SAVE_NEXT(next_save);
            }
#endif
        }
        x0 = lo2(X);
        y0 = lo2(Y);
        x1 = hi2(X);
        y1 = hi2(Y);
        n0 = n;
        n1 = n;
#if MANDEL_PERIODIC
        if (done0) n0 = cap;  // mandel_finish returns the cap at once
        if (done1) n1 = cap;
#endif
    }
    Cnt2 r;
    r.n0 = (n0 < p) ? n0 : mandel_finish<MANDEL_B>(c.re0, c.im0, x0, y0, n0, cap);
    r.n1 = (n1 < p) ? n1 : mandel_finish<MANDEL_B>(c.re1, c.im1, x1, y1, n1, cap);
    return r;
}
