// EXPERIMENT (tools/mandel_parts_probe.py): persistent warps with dynamic
// warp-granular tasks, appended to mandelbrot_blocked.cu.  A void index Map
// over nthreads = one resident wave; each warp takes the next task of 32
// consecutive pixels from ctr[0] until the image is done; the last warp to
// finish resets both counters (graph replays start from zero).
void mandel_dyn(unsigned i, const Pos *pos, int *out, unsigned *ctr, unsigned n, unsigned nwarps, int cap) {
    const unsigned lane = threadIdx.x & 31u;
    for (;;) {
        unsigned t = 0;
        if (lane == 0) t = atomicAdd(&ctr[0], 1u);
        t = __shfl_sync(0xffffffffu, t, 0);
        const unsigned long long p0 = (unsigned long long)t * 32u;
        if (p0 >= n) break;
        const unsigned long long px = p0 + lane;
        if (px < n) out[px] = mandelbrot_blocked(pos[px], cap);
    }
    __syncwarp();
    if (lane == 0) {
        __threadfence();
        const unsigned d = atomicAdd(&ctr[1], 1u);
        if (d == nwarps - 1) {
            ctr[0] = 0;
            ctr[1] = 0;
            __threadfence();
        }
    }
}
