// builtin.cu -- helper kernels of libskel compiled ahead of time by nvcc for
// sm_100a (the skeleton kernels themselves are generated at run time by NVRTC).
//
//  * fill:    device-side initialisation of a vector with one element value
//  * combine: element-wise merge of the per-device copies of a copy-distributed
//             vector (Listing 4, "reduce (element-wise add) all
//             copies"), used when the logical devices live in this process
//             (skel_init); in one-process-per-GPU mode NCCL does this.
#include <cstdint>

#include "internal.h"

namespace {

constexpr int kMaxSrc = 64;
struct SrcList {
    const void *p[kMaxSrc];
};

__global__ void fill_u32_kernel(uint32_t *dst, size_t n, uint32_t v) {
    const size_t stride = (size_t)gridDim.x * blockDim.x;
    for (size_t i = (size_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) dst[i] = v;
}
__global__ void fill_u32x4_kernel(uint4 *dst, size_t n4, uint32_t v) {
    const size_t stride = (size_t)gridDim.x * blockDim.x;
    const uint4 q = make_uint4(v, v, v, v);
    for (size_t i = (size_t)blockIdx.x * blockDim.x + threadIdx.x; i < n4; i += stride) dst[i] = q;
}
__global__ void fill_bytes_kernel(unsigned char *dst, size_t n, const unsigned char *__restrict__ pat, size_t es,
                                  uint4 inl0, uint4 inl1, uint4 inl2, uint4 inl3) {
    unsigned char local[64];
    const uint4 q[4] = {inl0, inl1, inl2, inl3};
    memcpy(local, q, 64);
    const size_t stride = (size_t)gridDim.x * blockDim.x;
    for (size_t i = (size_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride)
        for (size_t b = 0; b < es; ++b) dst[i * es + b] = local[b];
}

template <class T, int OP> __device__ __forceinline__ T apply(T a, T b) {
    if (OP == SKEL_COMBINE_ADD) return a + b;
    if (OP == SKEL_COMBINE_MIN) return b < a ? b : a;
    if (OP == SKEL_COMBINE_MAX) return a < b ? b : a;
    return a * b;
}

template <class T, int OP>
__global__ void combine_kernel(T *dst, SrcList srcs, int nsrc, size_t count) {
    const size_t stride = (size_t)gridDim.x * blockDim.x;
    for (size_t i = (size_t)blockIdx.x * blockDim.x + threadIdx.x; i < count; i += stride) {
        T acc = static_cast<const T *>(srcs.p[0])[i];
        for (int j = 1; j < nsrc; ++j) acc = apply<T, OP>(acc, static_cast<const T *>(srcs.p[j])[i]);
        dst[i] = acc;
    }
}
// 4-byte types, all pointers 16-byte aligned: 128-bit loads/stores
template <class T, int OP>
__global__ void combine4_kernel(T *dst, SrcList srcs, int nsrc, size_t count4) {
    const size_t stride = (size_t)gridDim.x * blockDim.x;
    for (size_t i = (size_t)blockIdx.x * blockDim.x + threadIdx.x; i < count4; i += stride) {
        uint4 q = __ldcs(static_cast<const uint4 *>(srcs.p[0]) + i);
        T a[4];
        memcpy(a, &q, 16);
        for (int j = 1; j < nsrc; ++j) {
            uint4 r = __ldcs(static_cast<const uint4 *>(srcs.p[j]) + i);
            T b[4];
            memcpy(b, &r, 16);
#pragma unroll
            for (int e = 0; e < 4; ++e) a[e] = apply<T, OP>(a[e], b[e]);
        }
        memcpy(&q, a, 16);
        __stcs(reinterpret_cast<uint4 *>(dst) + i, q);
    }
}

int grid_for(size_t work, int block) {
    int dev = 0, sms = 148;
    cudaGetDevice(&dev);
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    size_t g = (work + block - 1) / block;
    const size_t cap = (size_t)sms * (2048 / block) * 4;
    if (g > cap) g = cap;
    if (g < 1) g = 1;
    return (int)g;
}

template <class T, int OP>
cudaError_t combine_t(void *dst, const void *const *srcs, int nsrc, size_t count, cudaStream_t s) {
    SrcList l{};
    bool al = (reinterpret_cast<uintptr_t>(dst) & 15) == 0;
    for (int j = 0; j < nsrc; ++j) {
        l.p[j] = srcs[j];
        al = al && (reinterpret_cast<uintptr_t>(srcs[j]) & 15) == 0;
    }
    const int block = 256;
    if (sizeof(T) == 4 && al) {
        const size_t c4 = count / 4;
        if (c4) combine4_kernel<T, OP><<<grid_for(c4, block), block, 0, s>>>(static_cast<T *>(dst), l, nsrc, c4);
        const size_t done = c4 * 4;
        if (count > done) {
            SrcList t{};
            for (int j = 0; j < nsrc; ++j) t.p[j] = static_cast<const T *>(srcs[j]) + done;
            combine_kernel<T, OP><<<1, block, 0, s>>>(static_cast<T *>(dst) + done, t, nsrc, count - done);
        }
    } else {
        combine_kernel<T, OP><<<grid_for(count, block), block, 0, s>>>(static_cast<T *>(dst), l, nsrc, count);
    }
    return cudaGetLastError();
}

template <class T>
cudaError_t combine_op(void *dst, const void *const *srcs, int nsrc, size_t count, skel_combine op, cudaStream_t s) {
    switch (op) {
        case SKEL_COMBINE_ADD: return combine_t<T, SKEL_COMBINE_ADD>(dst, srcs, nsrc, count, s);
        case SKEL_COMBINE_MIN: return combine_t<T, SKEL_COMBINE_MIN>(dst, srcs, nsrc, count, s);
        case SKEL_COMBINE_MAX: return combine_t<T, SKEL_COMBINE_MAX>(dst, srcs, nsrc, count, s);
        case SKEL_COMBINE_PROD: return combine_t<T, SKEL_COMBINE_PROD>(dst, srcs, nsrc, count, s);
        default: return cudaErrorInvalidValue;
    }
}

// dst[j*bytes .. (j+1)*bytes) = srcs[j][0 .. bytes): collects the per-device
// partial results of Reduce/Scan (all pointers live in this process)
__global__ void gather_kernel(unsigned char *dst, SrcList srcs, int nsrc, size_t bytes) {
    for (size_t i = threadIdx.x; i < (size_t)nsrc * bytes; i += blockDim.x) {
        const int j = (int)(i / bytes);
        dst[i] = static_cast<const unsigned char *>(srcs.p[j])[i - j * bytes];
    }
}

}  // namespace

namespace skelrt {

cudaError_t launch_gather(void *dst, const void *const *srcs, int nsrc, size_t bytes, cudaStream_t s) {
    if (nsrc < 1 || nsrc > kMaxSrc) return cudaErrorInvalidValue;
    SrcList l{};
    for (int j = 0; j < nsrc; ++j) l.p[j] = srcs[j];
    gather_kernel<<<1, 256, 0, s>>>(static_cast<unsigned char *>(dst), l, nsrc, bytes);
    return cudaGetLastError();
}

cudaError_t launch_fill(void *dst, size_t n, const void *elem, size_t es, cudaStream_t s) {
    if (n == 0) return cudaSuccess;
    if (es > 64) return cudaErrorInvalidValue;
    unsigned char pat[64] = {0};
    memcpy(pat, elem, es);
    const int block = 256;
    bool uniform4 = (es % 4 == 0);
    uint32_t w0 = 0;
    memcpy(&w0, pat, 4);
    for (size_t b = 0; uniform4 && b < es; b += 4) uniform4 = memcmp(pat + b, &w0, 4) == 0;
    if (uniform4) {
        const size_t words = n * es / 4;
        if ((reinterpret_cast<uintptr_t>(dst) & 15) == 0 && words >= 4) {
            const size_t n4 = words / 4;
            fill_u32x4_kernel<<<grid_for(n4, block), block, 0, s>>>(static_cast<uint4 *>(dst), n4, w0);
            if (words > n4 * 4)
                fill_u32_kernel<<<1, block, 0, s>>>(static_cast<uint32_t *>(dst) + n4 * 4, words - n4 * 4, w0);
        } else {
            fill_u32_kernel<<<grid_for(words, block), block, 0, s>>>(static_cast<uint32_t *>(dst), words, w0);
        }
    } else {
        uint4 q[4];
        memcpy(q, pat, 64);
        fill_bytes_kernel<<<grid_for(n, block), block, 0, s>>>(static_cast<unsigned char *>(dst), n, nullptr, es, q[0],
                                                               q[1], q[2], q[3]);
    }
    return cudaGetLastError();
}

cudaError_t launch_combine(void *dst, const void *const *srcs, int nsrc, size_t count, skel_dtype dt,
                           skel_combine op, cudaStream_t s) {
    if (count == 0) return cudaSuccess;
    if (nsrc < 1 || nsrc > kMaxSrc) return cudaErrorInvalidValue;
    switch (dt) {
        case SKEL_DT_F32: return combine_op<float>(dst, srcs, nsrc, count, op, s);
        case SKEL_DT_F64: return combine_op<double>(dst, srcs, nsrc, count, op, s);
        case SKEL_DT_I32: return combine_op<int32_t>(dst, srcs, nsrc, count, op, s);
        case SKEL_DT_U32: return combine_op<uint32_t>(dst, srcs, nsrc, count, op, s);
        case SKEL_DT_I64: return combine_op<long long>(dst, srcs, nsrc, count, op, s);
        case SKEL_DT_U64: return combine_op<unsigned long long>(dst, srcs, nsrc, count, op, s);
        default: return cudaErrorInvalidValue;
    }
}

}  // namespace skelrt
