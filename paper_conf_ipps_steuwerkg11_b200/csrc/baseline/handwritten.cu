// handwritten.cu -- the same four operations written directly in CUDA C++
// and compiled ahead of time by nvcc, as a programmer would without the
// skeleton library.  Measurement only (the analog of
// PAPER.md's "SkelCL vs OpenCL" overhead): bench.py
// times these beside the NVRTC-injected skeletons on the same buffers.
// Element-wise kernels use the usual float4 grid-stride loop; the reduction
// is the usual block-reduce + atomicAdd; the scan is CUB's DeviceScan (the
// library a CUDA programmer would reach for).
#include <cub/cub.cuh>
#include <cuda_runtime.h>

namespace {
__global__ void hw_map(const float4 *__restrict__ x, float4 *__restrict__ y, size_t n4) {
    for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n4; i += (size_t)gridDim.x * blockDim.x) {
        float4 v = x[i];
        v.x = __fadd_rn(__fmul_rn(v.x, 2.0f), 1.0f);
        v.y = __fadd_rn(__fmul_rn(v.y, 2.0f), 1.0f);
        v.z = __fadd_rn(__fmul_rn(v.z, 2.0f), 1.0f);
        v.w = __fadd_rn(__fmul_rn(v.w, 2.0f), 1.0f);
        y[i] = v;
    }
}
__global__ void hw_saxpy(const float4 *__restrict__ x, const float4 *__restrict__ y, float4 *__restrict__ z, float a,
                         size_t n4) {
    for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n4; i += (size_t)gridDim.x * blockDim.x) {
        const float4 u = x[i], v = y[i];
        z[i] = make_float4(__fadd_rn(__fmul_rn(a, u.x), v.x), __fadd_rn(__fmul_rn(a, u.y), v.y),
                           __fadd_rn(__fmul_rn(a, u.z), v.z), __fadd_rn(__fmul_rn(a, u.w), v.w));
    }
}
__global__ void hw_sum(const float4 *__restrict__ x, size_t n4, float *out) {
    float s = 0.0f;
    for (size_t i = blockIdx.x * (size_t)blockDim.x + threadIdx.x; i < n4; i += (size_t)gridDim.x * blockDim.x) {
        const float4 v = x[i];
        s += (v.x + v.y) + (v.z + v.w);
    }
    typedef cub::BlockReduce<float, 256> BR;
    __shared__ typename BR::TempStorage tmp;
    const float b = BR(tmp).Sum(s);
    if (threadIdx.x == 0) atomicAdd(out, b);
}
int grid(size_t n4) {
    int dev = 0, sms = 148;
    cudaGetDevice(&dev);
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    size_t g = (n4 + 255) / 256, cap = (size_t)sms * 8 * 4;
    return (int)(g < cap ? (g ? g : 1) : cap);
}
}  // namespace

extern "C" {
// n must be a multiple of 4 (float4 loops); all pointers are device pointers
int hw_map_f32(const float *x, float *y, size_t n, void *stream) {
    hw_map<<<grid(n / 4), 256, 0, (cudaStream_t)stream>>>((const float4 *)x, (float4 *)y, n / 4);
    return (int)cudaGetLastError();
}
int hw_saxpy_f32(const float *x, const float *y, float *z, float a, size_t n, void *stream) {
    hw_saxpy<<<grid(n / 4), 256, 0, (cudaStream_t)stream>>>((const float4 *)x, (const float4 *)y, (float4 *)z, a, n / 4);
    return (int)cudaGetLastError();
}
int hw_sum_f32(const float *x, size_t n, float *out, void *stream) {
    cudaMemsetAsync(out, 0, sizeof(float), (cudaStream_t)stream);
    hw_sum<<<grid(n / 4), 256, 0, (cudaStream_t)stream>>>((const float4 *)x, n / 4, out);
    return (int)cudaGetLastError();
}
// CUB exclusive sum; temp storage is allocated on first use and kept
int hw_exscan_f32(const float *x, float *y, size_t n, void *stream) {
    static void *tmp = nullptr;
    static size_t tmp_bytes = 0;
    size_t need = 0;
    cub::DeviceScan::ExclusiveSum(nullptr, need, x, y, (int64_t)n, (cudaStream_t)stream);
    if (need > tmp_bytes) {
        if (tmp) cudaFree(tmp);
        cudaMalloc(&tmp, need);
        tmp_bytes = need;
    }
    cub::DeviceScan::ExclusiveSum(tmp, tmp_bytes, x, y, (int64_t)n, (cudaStream_t)stream);
    return (int)cudaGetLastError();
}
}

// CUB's two-kernel DeviceReduce::Sum (small-size comparison, tools/small_n_probe.py)
extern "C" int hw_cubsum_f32(const float *x, size_t n, float *out, void *stream) {
    static void *tmp = nullptr;
    static size_t tmp_bytes = 0;
    size_t need = 0;
    cub::DeviceReduce::Sum(nullptr, need, x, out, (int64_t)n, (cudaStream_t)stream);
    if (need > tmp_bytes) {
        if (tmp) cudaFree(tmp);
        cudaMalloc(&tmp, need);
        tmp_bytes = need;
    }
    cub::DeviceReduce::Sum(tmp, tmp_bytes, x, out, (int64_t)n, (cudaStream_t)stream);
    return (int)cudaGetLastError();
}
