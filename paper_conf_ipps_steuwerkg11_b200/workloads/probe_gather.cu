// Gather probe (see probe_scatter.cu): PROBE_K scattered 4-byte loads per
// element from an image-sized buffer, summed so that none is dead.
#define PROBE_K 64
static __forceinline__ unsigned probe_hash(unsigned x) {
    x ^= x >> 16;
    x *= 0x7feb352du;
    x ^= x >> 15;
    x *= 0x846ca68bu;
    x ^= x >> 16;
    return x;
}
float probe_gather(unsigned i, const float *f, unsigned nvox) {
    float acc = 0.0f;
#pragma unroll 8
    for (int k = 0; k < PROBE_K; ++k) acc += __ldg(&f[probe_hash(i * PROBE_K + k) % nvox]);
    return acc;
}
