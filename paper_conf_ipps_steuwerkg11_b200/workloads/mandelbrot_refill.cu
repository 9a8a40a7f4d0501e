
// ---- persistent warps with pixel refill, appended to
// mandelbrot_blocked.cu.  A void index Map over a fixed number of threads
// (about one resident wave); each warp keeps its 32 lanes busy: a lane whose
// pixel has finished takes the next unprocessed pixel from a global counter
// (one atomic per warp and refill, row-major order, so the lanes of a warp
// write neighbouring counts), instead of idling until the warp's slowest pixel
// is done (the 8% of lane slots a one-pixel-per-thread Map loses on the
// paper's image, plus the blocks its escaping lanes wait through).  Every
// pixel is iterated with exactly the operations of eq. (5) as written (the
// blocked scheme with roll-back of mandelbrot_blocked.cu: 8 updates per block,
// an escape inside a block replays it update by update), so the counts are
// bit-identical; with MANDEL_PERIODIC each pixel also stops when its orbit
// repeats bit for bit (Brent's schedule per pixel).
//   img      row-major int32 image (a vector argument, written by side effect)
//   next_pix a one-int vector holding 0 before the launch (the work counter)
#ifndef MANDEL_RB
#define MANDEL_RB 8
#endif
#ifndef MANDEL_CHUNK
#define MANDEL_CHUNK 256  // pixels a warp takes from the global counter at a time
#endif
void mandelbrot_refill(unsigned i, int *img, int *next_pix, int width, int height, int cap) {
    (void)i;
    const unsigned FULL = 0xffffffffu;
    const int lane = (int)(threadIdx.x & 31u);
    const int total = width * height;
    int q_next = 0, q_end = 0;  // the warp's queue of pixels [q_next, q_end) (warp-uniform)
    bool exhausted = false;     // the global counter has passed the last pixel (warp-uniform)
    int pix = -1;               // this lane's pixel, -1: none
    float x = 0.0f, y = 0.0f, cr = 0.0f, ci = 0.0f;
    int n = 0;
#if MANDEL_PERIODIC
    unsigned svx = 0u, svy = 0u;
    int blk = 0, next_save = 1;
#endif
    for (;;) {
        const unsigned need = __ballot_sync(FULL, pix < 0);
        if (need && !(exhausted && q_next >= q_end)) {
            if (q_next >= q_end) {  // refill the warp's queue
                int b = 0;
                if (lane == 0) b = atomicAdd(next_pix, MANDEL_CHUNK);
                b = __shfl_sync(FULL, b, 0);
                q_next = b < total ? b : total;
                q_end = b + MANDEL_CHUNK < total ? b + MANDEL_CHUNK : total;
                exhausted = b + MANDEL_CHUNK >= total;
            }
            const int r = __popc(need & ((1u << lane) - 1u));
            if (pix < 0 && q_next + r < q_end) {
                pix = q_next + r;
                const int px = pix % width, py = pix / width;
                cr = (float)(-2.5 + (double)px * (4.0 / (double)width));
                ci = (float)(-1.5 + (double)py * (3.0 / (double)height));
                x = 0.0f;
                y = 0.0f;
                n = 0;
#if MANDEL_PERIODIC
                svx = mandel_bits(x);
                svy = mandel_bits(y);
                blk = 0;
                next_save = 1;
#endif
            }
            const int took = __popc(need) < q_end - q_next ? __popc(need) : q_end - q_next;
            q_next += took;
        }
        const bool has = pix >= 0;
        if (!__any_sync(FULL, has) && exhausted && q_next >= q_end) break;
        if (has) {
            bool done = false;
            if (n + MANDEL_RB <= cap) {
                const float x0 = x, y0 = y;
                bool out = false;
#pragma unroll
                for (int k = 0; k < MANDEL_RB; ++k) {
                    const float xx = x * x, yy = y * y;
                    out = out | !(xx + yy <= 4.0f);
                    const float xt = (xx - yy) + cr;
                    y = (2.0f * x) * y + ci;
                    x = xt;
                }
                if (out) {  // escaped inside this block: replay it update by update
                    x = x0;
                    y = y0;
                    while (n < cap && x * x + y * y <= 4.0f) {
                        const float xt = (x * x - y * y) + cr;
                        y = (2.0f * x) * y + ci;
                        x = xt;
                        ++n;
                    }
                    done = true;
                } else {
                    n += MANDEL_RB;
#if MANDEL_PERIODIC
                    if (mandel_bits(x) == svx && mandel_bits(y) == svy) {  // exact cycle: a member
                        n = cap;
                    } else if (++blk == next_save) {
                        svx = mandel_bits(x);
                        svy = mandel_bits(y);
                        next_save <<= 1;
                    }
#endif
                    done = n >= cap;
                }
            } else {  // fewer than a block of updates left before the cap
                while (n < cap && x * x + y * y <= 4.0f) {
                    const float xt = (x * x - y * y) + cr;
                    y = (2.0f * x) * y + ci;
                    x = xt;
                    ++n;
                }
                done = true;
            }
            if (done) {
                img[pix] = n;
                pix = -1;
            }
        }
    }
}
