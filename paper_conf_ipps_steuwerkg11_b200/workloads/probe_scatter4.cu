// Vector-reduction probe (see probe_scatter.cu): PROBE_K red.global.add.v4.f32
// per element at random 16-byte aligned addresses of an image-sized buffer --
// the request the LM OSEM back projection issues per 4-float group.
#define PROBE_K 64
static __forceinline__ unsigned probe_hash(unsigned x) {
    x ^= x >> 16;
    x *= 0x7feb352du;
    x ^= x >> 15;
    x *= 0x846ca68bu;
    x ^= x >> 16;
    return x;
}
static __forceinline__ void probe_red4(float *p, float v) {
    asm volatile("red.global.add.v4.f32 [%0], {%1, %1, %1, %1};" ::"l"(p), "f"(v) : "memory");
}
void probe_scatter_red4(unsigned i, float *c, unsigned nvox) {
#pragma unroll 8
    for (int k = 0; k < PROBE_K; ++k) probe_red4(&c[(probe_hash(i * PROBE_K + k) % nvox) & ~3u], 1.0f);
}
