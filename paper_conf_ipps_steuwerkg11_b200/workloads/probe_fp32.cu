// FP32 lane-peak probe (measurement only): the denominator of the Mandelbrot
// roofline, measured in the same bench run.  An index Map whose every thread
// runs PROBE_FP32_CHAINS independent dependency chains of packed two-lane
// adds (add.rn.f32x2 -> SASS FADD2: one instruction, two FP32 operations per
// lane) for `iters` steps; 2 * PROBE_FP32_CHAINS * iters FP32 operations per
// element.  On B200 the packed and the scalar forms both saturate the FMA
// pipes at ~128 FP32 operations per SM and cycle (tools/fp32_probe.cu).
#define PROBE_FP32_CHAINS 8
float probe_fp32(unsigned i, float b, int iters) {
    unsigned long long a[PROBE_FP32_CHAINS];
    const unsigned long long bb = ((unsigned long long)__float_as_uint(b) << 32) | __float_as_uint(b);
#pragma unroll
    for (int j = 0; j < PROBE_FP32_CHAINS; ++j) {
        const float v = (float)(i & 1023u) * 1e-3f + (float)j;
        a[j] = ((unsigned long long)__float_as_uint(v) << 32) | __float_as_uint(v);
    }
    // 16 steps per trip: the loop's counter, compare and branch take issue slots
    // the FADD2s (two cycles of the FMA pipes each) leave free
#pragma unroll 16
    for (int k = 0; k < iters; ++k) {
#pragma unroll
        for (int j = 0; j < PROBE_FP32_CHAINS; ++j)
            asm volatile("add.rn.f32x2 %0, %1, %2;" : "=l"(a[j]) : "l"(a[j]), "l"(bb));
    }
    unsigned long long s = 0;
#pragma unroll
    for (int j = 0; j < PROBE_FP32_CHAINS; ++j) s ^= a[j];
    return __uint_as_float((unsigned)(s ^ (s >> 32)));
}
