// FP32 issue/pipe throughput probe for the Mandelbrot roofline (B200, sm_100a).
// Standalone: nvcc -gencode arch=compute_100a,code=sm_100a -O3 -fmad=false
//             -o /tmp/fp32_probe tools/fp32_probe.cu && /tmp/fp32_probe
// Each kernel runs NCH independent dependency chains per thread over ITER
// iterations on a full grid; ops are counted per lane (a packed f32x2
// instruction counts 2).  The SM clock is measured in-kernel (clock64 against
// globaltimer), so the result is lane-ops per SM per cycle: 128 = one FP32
// warp instruction per SMSP per cycle.
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

#define NCH 8
#define ITER 4096

__device__ unsigned long long g_c0, g_c1, g_t0, g_t1;

__device__ __forceinline__ void clk_begin() {
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        unsigned long long t;
        asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
        g_t0 = t;
        g_c0 = clock64();
    }
}
__device__ __forceinline__ void clk_end() {
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        unsigned long long t;
        asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
        g_t1 = t;
        g_c1 = clock64();
    }
}

// 1: FADD r,r,r
__global__ void k_fadd(float *out, float b) {
    clk_begin();
    float a[NCH];
#pragma unroll
    for (int j = 0; j < NCH; ++j) a[j] = threadIdx.x * 1e-7f + j;
    for (int i = 0; i < ITER; ++i) {
#pragma unroll
        for (int j = 0; j < NCH; ++j) a[j] = a[j] + b;
    }
    float s = 0;
#pragma unroll
    for (int j = 0; j < NCH; ++j) s += a[j];
    clk_end();
    if (s == 1234.5f) out[0] = s;
}
// 2: FMUL r,r,r
__global__ void k_fmul(float *out, float b) {
    clk_begin();
    float a[NCH];
#pragma unroll
    for (int j = 0; j < NCH; ++j) a[j] = threadIdx.x * 1e-7f + j;
    for (int i = 0; i < ITER; ++i) {
#pragma unroll
        for (int j = 0; j < NCH; ++j) a[j] = a[j] * b;
    }
    float s = 0;
#pragma unroll
    for (int j = 0; j < NCH; ++j) s += a[j];
    clk_end();
    if (s == 1234.5f) out[0] = s;
}
// 3: FFMA r,r,r,r
__global__ void k_ffma(float *out, float b, float c) {
    clk_begin();
    float a[NCH];
#pragma unroll
    for (int j = 0; j < NCH; ++j) a[j] = threadIdx.x * 1e-7f + j;
    for (int i = 0; i < ITER; ++i) {
#pragma unroll
        for (int j = 0; j < NCH; ++j) a[j] = __fmaf_rn(a[j], b, c);
    }
    float s = 0;
#pragma unroll
    for (int j = 0; j < NCH; ++j) s += a[j];
    clk_end();
    if (s == 1234.5f) out[0] = s;
}
typedef unsigned long long f2;
__device__ __forceinline__ f2 add2(f2 a, f2 b) {
    f2 d;
    asm volatile("add.rn.f32x2 %0, %1, %2;" : "=l"(d) : "l"(a), "l"(b));
    return d;
}
__device__ __forceinline__ f2 fma2(f2 a, f2 b, f2 c) {
    f2 d;
    asm volatile("fma.rn.f32x2 %0, %1, %2, %3;" : "=l"(d) : "l"(a), "l"(b), "l"(c));
    return d;
}
// 4: FADD2 (packed)
__global__ void k_fadd2(float *out, float b) {
    clk_begin();
    f2 a[NCH];
    const f2 bb = ((f2)__float_as_uint(b) << 32) | __float_as_uint(b);
#pragma unroll
    for (int j = 0; j < NCH; ++j) a[j] = (f2)(threadIdx.x + j);
    for (int i = 0; i < ITER; ++i) {
#pragma unroll
        for (int j = 0; j < NCH; ++j) a[j] = add2(a[j], bb);
    }
    f2 s = 0;
#pragma unroll
    for (int j = 0; j < NCH; ++j) s ^= a[j];
    clk_end();
    if (s == 12345) out[0] = 1;
}
// 5: FFMA2 (packed)
__global__ void k_ffma2(float *out, float b, float c) {
    clk_begin();
    f2 a[NCH];
    const f2 bb = ((f2)__float_as_uint(b) << 32) | __float_as_uint(b);
    const f2 cc = ((f2)__float_as_uint(c) << 32) | __float_as_uint(c);
#pragma unroll
    for (int j = 0; j < NCH; ++j) a[j] = (f2)(threadIdx.x + j);
    for (int i = 0; i < ITER; ++i) {
#pragma unroll
        for (int j = 0; j < NCH; ++j) a[j] = fma2(a[j], bb, cc);
    }
    f2 s = 0;
#pragma unroll
    for (int j = 0; j < NCH; ++j) s ^= a[j];
    clk_end();
    if (s == 12345) out[0] = 1;
}
// 6: FADD + FSETP accumulate (escape-test shape)
__global__ void k_fadd_fsetp(float *out, float b) {
    clk_begin();
    float a[NCH];
    bool o = false;
#pragma unroll
    for (int j = 0; j < NCH; ++j) a[j] = threadIdx.x * 1e-7f + j;
    for (int i = 0; i < ITER; ++i) {
#pragma unroll
        for (int j = 0; j < NCH; ++j) {
            a[j] = a[j] + b;
            o = o | !(a[j] <= 4.0e30f);
        }
    }
    float s = 0;
#pragma unroll
    for (int j = 0; j < NCH; ++j) s += a[j];
    clk_end();
    if (s == 1234.5f || o) out[0] = s;
}
// 7: Mandelbrot member block: c inside the main cardioid, 4 independent pixels
// per thread (ILP), 8 FP32 + 1 FSETP per update, no loop exit (ITER updates)
__global__ void k_mandel(float *out, float cr) {
    clk_begin();
    float x[4], y[4], ci[4];
    bool o = false;
#pragma unroll
    for (int j = 0; j < 4; ++j) { x[j] = 0; y[j] = 0; ci[j] = 0.01f * j + threadIdx.x * 1e-6f; }
    for (int i = 0; i < ITER / 4; ++i) {
#pragma unroll
        for (int j = 0; j < 4; ++j) {
            const float xx = x[j] * x[j], yy = y[j] * y[j];
            o = o | !(xx + yy <= 4.0f);
            const float xt = (xx - yy) + cr;
            y[j] = (2.0f * x[j]) * y[j] + ci[j];
            x[j] = xt;
        }
    }
    float s = 0;
#pragma unroll
    for (int j = 0; j < 4; ++j) s += x[j] + y[j];
    clk_end();
    if (s == 1234.5f || o) out[0] = s;
}
// 8: the same, no escape test (7 FP32 per update)
__global__ void k_mandel_notest(float *out, float cr) {
    clk_begin();
    float x[4], y[4], ci[4];
#pragma unroll
    for (int j = 0; j < 4; ++j) { x[j] = 0; y[j] = 0; ci[j] = 0.01f * j + threadIdx.x * 1e-6f; }
    for (int i = 0; i < ITER / 4; ++i) {
#pragma unroll
        for (int j = 0; j < 4; ++j) {
            const float xx = x[j] * x[j], yy = y[j] * y[j];
            const float xt = (xx - yy) + cr;
            y[j] = (2.0f * x[j]) * y[j] + ci[j];
            x[j] = xt;
        }
    }
    float s = 0;
#pragma unroll
    for (int j = 0; j < 4; ++j) s += x[j] + y[j];
    clk_end();
    if (s == 1234.5f) out[0] = s;
}
// 9: x+x instead of 2*x (FADD r,r instead of FMUL imm)
__global__ void k_mandel_xx(float *out, float cr) {
    clk_begin();
    float x[4], y[4], ci[4];
    bool o = false;
#pragma unroll
    for (int j = 0; j < 4; ++j) { x[j] = 0; y[j] = 0; ci[j] = 0.01f * j + threadIdx.x * 1e-6f; }
    for (int i = 0; i < ITER / 4; ++i) {
#pragma unroll
        for (int j = 0; j < 4; ++j) {
            const float xx = x[j] * x[j], yy = y[j] * y[j];
            o = o | !(xx + yy <= 4.0f);
            const float xt = (xx - yy) + cr;
            y[j] = (x[j] + x[j]) * y[j] + ci[j];
            x[j] = xt;
        }
    }
    float s = 0;
#pragma unroll
    for (int j = 0; j < 4; ++j) s += x[j] + y[j];
    clk_end();
    if (s == 1234.5f || o) out[0] = s;
}


// 10: scalar member loop, escape test accumulated with FMNMX (m = max(m, s))
__global__ void k_mandel_max(float *out, float cr) {
    clk_begin();
    float x[4], y[4], ci[4], m[4];
#pragma unroll
    for (int j = 0; j < 4; ++j) { x[j] = 0; y[j] = 0; m[j] = 0; ci[j] = 0.01f * j + threadIdx.x * 1e-6f; }
    for (int i = 0; i < ITER / 4; ++i) {
#pragma unroll
        for (int j = 0; j < 4; ++j) {
            const float xx = x[j] * x[j], yy = y[j] * y[j];
            m[j] = fmaxf(m[j], xx + yy);
            const float xt = (xx - yy) + cr;
            y[j] = (2.0f * x[j]) * y[j] + ci[j];
            x[j] = xt;
        }
    }
    float s = 0;
#pragma unroll
    for (int j = 0; j < 4; ++j) s += x[j] + y[j] + m[j];
    clk_end();
    if (s == 1234.5f) out[0] = s;
}
__device__ __forceinline__ f2 mul2z(f2 a, f2 b, f2 nz) { return fma2(a, b, nz); }
__device__ __forceinline__ f2 sub2(f2 a, f2 b) {
    f2 d;
    asm volatile("sub.rn.f32x2 %0, %1, %2;" : "=l"(d) : "l"(a), "l"(b));
    return d;
}
__device__ __forceinline__ f2 mk2(float lo, float hi) { return ((f2)__float_as_uint(hi) << 32) | __float_as_uint(lo); }
__device__ __forceinline__ float lo2(f2 v) { return __uint_as_float((unsigned)v); }
__device__ __forceinline__ float hi2(f2 v) { return __uint_as_float((unsigned)(v >> 32)); }
__device__ f2 g_nz = 0x8000000080000000ull;
// 11..13: packed pair member loop, 2 pairs per thread; test: 0 none, 1 FSETP.OR, 2 FMNMX
template <int TEST>
__global__ void k_pairs(float *out, float cr0) {
    clk_begin();
    const f2 nz = *(volatile f2 *)&g_nz;
    f2 X[2], Y[2], CI[2];
    const f2 CR = mk2(cr0, cr0);
    bool o = false;
    float m = 0.f;
#pragma unroll
    for (int j = 0; j < 2; ++j) { X[j] = 0; Y[j] = 0; CI[j] = mk2(0.01f * j + threadIdx.x * 1e-6f, 0.02f * j); }
    for (int i = 0; i < ITER / 4; ++i) {
#pragma unroll
        for (int j = 0; j < 2; ++j) {
            const f2 XX = mul2z(X[j], X[j], nz), YY = mul2z(Y[j], Y[j], nz);
            if (TEST) {
                const f2 S = add2(XX, YY);
                if (TEST == 1) { o = o | !(lo2(S) <= 4.0f); o = o | !(hi2(S) <= 4.0f); }
                else { m = fmaxf(m, lo2(S)); m = fmaxf(m, hi2(S)); }
            }
            const f2 XT = add2(sub2(XX, YY), CR);
            Y[j] = add2(mul2z(add2(X[j], X[j]), Y[j], nz), CI[j]);
            X[j] = XT;
        }
    }
    f2 s = 0;
#pragma unroll
    for (int j = 0; j < 2; ++j) s ^= X[j] ^ Y[j];
    clk_end();
    if (s == 12345 || o || m == 1234.5f) out[0] = 1;
}

// 14: scalar member loop, 4 pixels, tests folded pairwise with 3-input max (FMNMX3)
__global__ void k_mandel_max3(float *out, float cr) {
    clk_begin();
    float x[4], y[4], ci[4], s[4];
    float m = 0.f;
#pragma unroll
    for (int j = 0; j < 4; ++j) { x[j] = 0; y[j] = 0; ci[j] = 0.01f * j + threadIdx.x * 1e-6f; }
    for (int i = 0; i < ITER / 4; ++i) {
#pragma unroll
        for (int j = 0; j < 4; ++j) {
            const float xx = x[j] * x[j], yy = y[j] * y[j];
            s[j] = xx + yy;
            const float xt = (xx - yy) + cr;
            y[j] = (2.0f * x[j]) * y[j] + ci[j];
            x[j] = xt;
        }
        m = fmaxf(fmaxf(m, s[0]), s[1]);
        m = fmaxf(fmaxf(m, s[2]), s[3]);
    }
    float t = m;
#pragma unroll
    for (int j = 0; j < 4; ++j) t += x[j] + y[j];
    clk_end();
    if (t == 1234.5f) out[0] = t;
}

template <typename K, typename... A>
static void run(const char *name, double ops_per_thread_iter, K k, A... a) {
    float *out;
    cudaMalloc(&out, 4);
    int dev = 0, sms = 0;
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    const int threads = 256, blocks = sms * 8;  // 2048 threads per SM
    cudaEvent_t e0, e1;
    cudaEventCreate(&e0);
    cudaEventCreate(&e1);
    for (int w = 0; w < 3; ++w) k<<<blocks, threads>>>(out, a...);
    cudaEventRecord(e0);
    const int reps = 5;
    for (int r = 0; r < reps; ++r) k<<<blocks, threads>>>(out, a...);
    cudaEventRecord(e1);
    cudaEventSynchronize(e1);
    float ms;
    cudaEventElapsedTime(&ms, e0, e1);
    unsigned long long c0, c1, t0, t1;
    cudaMemcpyFromSymbol(&c0, g_c0, 8);
    cudaMemcpyFromSymbol(&c1, g_c1, 8);
    cudaMemcpyFromSymbol(&t0, g_t0, 8);
    cudaMemcpyFromSymbol(&t1, g_t1, 8);
    const double mhz = (double)(c1 - c0) / (double)(t1 - t0) * 1e3;
    const double ops = ops_per_thread_iter * (double)ITER * threads * blocks * reps;
    const double rate = ops / (ms * 1e-3);
    const double per_sm_clk = rate / (sms * mhz * 1e6);
    printf("%-16s %8.3f ms/launch  %7.2f T lane-ops/s  SM clock %6.0f MHz  %6.1f lane-ops/SM/clk\n", name,
           ms / reps, rate / 1e12, mhz, per_sm_clk);
    cudaFree(out);
    cudaError_t err = cudaGetLastError();
    if (err != cudaSuccess) printf("  error %s\n", cudaGetErrorString(err));
}

int main() {
    run("fadd", NCH, k_fadd, 1e-9f);
    run("fmul", NCH, k_fmul, 0.9999999f);
    run("ffma", NCH, k_ffma, 0.9999999f, 1e-9f);
    run("fadd2", 2 * NCH, k_fadd2, 1e-9f);
    run("ffma2", 2 * NCH, k_ffma2, 0.9999999f, 1e-9f);
    run("fadd+fsetp", NCH, k_fadd_fsetp, 1e-9f);   // FP32 ops only (FSETP not counted)
    run("mandel 8+1", 8.0, k_mandel, -0.1f);       // 8 FP32 per update as written
    run("mandel 7", 7.0, k_mandel_notest, -0.1f);  // 7 FP32 per update (test dropped)
    run("mandel x+x", 8.0, k_mandel_xx, -0.1f);
    run("mandel fmnmx", 8.0, k_mandel_max, -0.1f);
    run("mandel fmnmx3", 8.0, k_mandel_max3, -0.1f);
    run("pairs notest", 7.0, k_pairs<0>, -0.1f);  // per lane-update, 2 pairs x 2 pixels per iteration of 4 updates
    run("pairs fsetp", 8.0, k_pairs<1>, -0.1f);
    run("pairs fmnmx", 8.0, k_pairs<2>, -0.1f);
    return 0;
}
