// EXPERIMENT (tools/mandel_parts_probe.py): Mandelbrot with warp-local refill.
// A void index Map over one thread per lane of ceil(npix / MR_P) warps; warp w
// owns the MR_P consecutive pixels [w MR_P, (w+1) MR_P).  Every lane iterates
// blocks of 8 updates with the folded test and no replay (mandelbrot_blocked.cu
// MANDEL_NOREPLAY) and exact periodicity checking; a lane whose pixel is done
// stores the count and takes the warp's next pixel (rank among the finished
// lanes, no atomics), so the lanes of a warp stay busy until its backlog is
// exhausted.  c as the position vector (reading R5).
#ifndef MR_P
#define MR_P 256
#endif
static __forceinline__ float mr_max2(float a, float b) {
    float d;
    asm("max.NaN.f32 %0, %1, %2;" : "=f"(d) : "f"(a), "f"(b));
    return d;
}
void mandelbrot_refill(unsigned i, int *img, unsigned npix, int width, int height, int cap) {
    const unsigned lane = threadIdx.x & 31u;
    const unsigned base = (i >> 5) * (unsigned)MR_P;
    if (base >= npix) return;  // uniform across the warp
    const unsigned end = min(base + (unsigned)MR_P, npix);
    unsigned head = 32u;
    unsigned px = base + lane;
    bool act = px < end;
    float cr = 0.0f, ci = 0.0f, x = 0.0f, y = 0.0f;
    int n = 0, blk = 0, next_save = 1;
    unsigned sx = 0u, sy = 0u;
    auto init = [&](unsigned p) {
        const unsigned qx = p % (unsigned)width, qy = p / (unsigned)width;
        cr = (float)(-2.5 + (double)qx * (4.0 / (double)width));
        ci = (float)(-1.5 + (double)qy * (3.0 / (double)height));
        x = 0.0f;
        y = 0.0f;
        n = 0;
        blk = 0;
        next_save = 1;
        sx = __float_as_uint(x);
        sy = __float_as_uint(y);
    };
    if (act) init(px);
    while (__any_sync(0xffffffffu, act)) {
        int res = -1;
        if (act) {
            if (n + 8 <= cap) {
                float sv[8];
                float m = 0.0f;
#pragma unroll
                for (int k = 0; k < 8; ++k) {
                    const float xx = x * x, yy = y * y;
                    sv[k] = xx + yy;
                    const float xt = (xx - yy) + cr;
                    y = (2.0f * x) * y + ci;
                    x = xt;
                    if (k & 1) m = mr_max2(mr_max2(m, sv[k - 1]), sv[k]);
                }
                if (!(m <= 4.0f)) {
                    int k = 8;
#pragma unroll
                    for (int j = 7; j >= 0; --j)
                        if (!(sv[j] <= 4.0f)) k = j;
                    res = n + k;
                } else {
                    n += 8;
                    if (__float_as_uint(x) == sx && __float_as_uint(y) == sy) {
                        res = cap;  // exact cycle: a member
                    } else {
                        if (++blk == next_save) {
                            sx = __float_as_uint(x);
                            sy = __float_as_uint(y);
                            next_save <<= 1;
                        }
                        if (n >= cap) res = cap;
                    }
                }
            } else {  // the last cap mod 8 updates: the plain loop
                while (n < cap && x * x + y * y <= 4.0f) {
                    const float xt = (x * x - y * y) + cr;
                    y = (2.0f * x) * y + ci;
                    x = xt;
                    ++n;
                }
                res = n;
            }
        }
        const bool done = act && res >= 0;
        if (done) img[px] = res;
        const unsigned dm = __ballot_sync(0xffffffffu, done);
        if (done) {
            const unsigned np = base + head + __popc(dm & ((1u << lane) - 1u));
            if (np < end) {
                px = np;
                init(np);
            } else {
                act = false;
            }
        }
        head += __popc(dm);
    }
}
