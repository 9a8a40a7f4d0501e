// Roofline probes for the LM OSEM error-image Map (bench.py).
// The Siddon walk issues one scattered 4-byte request per voxel visit: a
// gather of f in the forward projection, a red.global.add.f32 into c in the
// back projection, and the 32 lanes of a warp are on 32 different rays, so
// every request of a warp instruction goes to a different L2 line.  These
// two Maps issue exactly that kind of request at random addresses of an
// image-sized (25 MB) buffer, PROBE_K per element, as fast as the hardware
// takes them: their request rates are the measured peaks the LM OSEM Map is
// compared with.
#define PROBE_K 64
static __forceinline__ unsigned probe_hash(unsigned x) {
    x ^= x >> 16;
    x *= 0x7feb352du;
    x ^= x >> 15;
    x *= 0x846ca68bu;
    x ^= x >> 16;
    return x;
}
static __forceinline__ void probe_red(float *p, float v) {
    asm volatile("red.global.add.f32 [%0], %1;" ::"l"(p), "f"(v) : "memory");
}
void probe_scatter_red(unsigned i, float *c, unsigned nvox) {
#pragma unroll 8
    for (int k = 0; k < PROBE_K; ++k) probe_red(&c[probe_hash(i * PROBE_K + k) % nvox], 1.0f);
}
