// scan_lab.cu -- stand-alone harness for the Scan skeleton kernel (lab tool,
// not part of the product).  Builds the Scan kernel around an unsigned +
// operator and launches it in isolation so that it can be timed, traced
// (-DSKEL_SCAN_TRACE) and checked:
//
//   nvcc -O2 -std=c++17 tools/scan_lab.cu -lnvrtc -lcuda -o scan_lab
//   ./scan_lab <skeletons dir> <log2n> <reps> [trace.bin] [-D... nvrtc options]
//
// The skeleton text is compiled with NVRTC exactly as libskel does
// (prelude + user function + "#define SKEL_FN" + red.cuh, -default-device).
// Check: out[0] == 0 and out[i+1] - out[i] == in[i] (mod 2^32) for every i,
// which is exactly the exclusive-scan definition (eq. (4)).
#include <cuda.h>
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <vector>

#include <nvrtc.h>

#include <fstream>
#include <sstream>
#include <string>

typedef unsigned long long skel_u64;
#define CKR(x)                                                                                   \
    do {                                                                                         \
        cudaError_t e_ = (x);                                                                    \
        if (e_ != cudaSuccess) {                                                                 \
            fprintf(stderr, "%s:%d %s: %s\n", __FILE__, __LINE__, #x, cudaGetErrorString(e_)); \
            exit(1);                                                                             \
        }                                                                                        \
    } while (0)

__global__ void lab_fill(unsigned *p, skel_u64 n) {
    for (skel_u64 i = blockIdx.x * (skel_u64)blockDim.x + threadIdx.x; i < n; i += (skel_u64)gridDim.x * blockDim.x)
        p[i] = (unsigned)((i * 0x9E3779B97F4A7C15ull) >> 61);  // 0..7
}
__global__ void lab_check(const unsigned *in, const unsigned *out, skel_u64 n, unsigned long long *bad) {
    for (skel_u64 i = blockIdx.x * (skel_u64)blockDim.x + threadIdx.x; i < n; i += (skel_u64)gridDim.x * blockDim.x) {
        const bool ok = i == 0 ? out[0] == 0u : out[i] - out[i - 1] == in[i - 1];
        if (!ok) atomicAdd(bad, 1ull);
    }
}

typedef CUresult (*PFN_encode)(CUtensorMap *, CUtensorMapDataType, cuuint32_t, void *, const cuuint64_t *,
                               const cuuint64_t *, const cuuint32_t *, const cuuint32_t *, CUtensorMapInterleave,
                               CUtensorMapSwizzle, CUtensorMapL2promotion, CUtensorMapFloatOOBfill);
static bool make_map(CUtensorMap *map, void *ptr, skel_u64 rows, unsigned box_rows) {
    static PFN_encode enc = nullptr;
    if (!enc) {
        void *p = nullptr;
        cudaDriverEntryPointQueryResult q;
        CKR(cudaGetDriverEntryPointByVersion("cuTensorMapEncodeTiled", &p, 12000, cudaEnableDefault, &q));
        enc = (PFN_encode)p;
    }
    cuuint64_t dims[2] = {32, rows};
    cuuint64_t strides[1] = {128};
    cuuint32_t box[2] = {32, box_rows};
    cuuint32_t estr[2] = {1, 1};
    return enc(map, CU_TENSOR_MAP_DATA_TYPE_UINT32, 2, ptr, dims, strides, box, estr, CU_TENSOR_MAP_INTERLEAVE_NONE,
               CU_TENSOR_MAP_SWIZZLE_128B, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
               CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE) == CUDA_SUCCESS;
}

#define CKD(x)                                                                       \
    do {                                                                             \
        CUresult r_ = (x);                                                           \
        if (r_ != CUDA_SUCCESS) {                                                    \
            const char *m_ = nullptr;                                                \
            cuGetErrorString(r_, &m_);                                               \
            fprintf(stderr, "%s:%d %s: %s\n", __FILE__, __LINE__, #x, m_ ? m_ : "?"); \
            exit(1);                                                                 \
        }                                                                            \
    } while (0)

static std::string slurp(const std::string &path) {
    std::ifstream f(path);
    if (!f) {
        fprintf(stderr, "cannot read %s\n", path.c_str());
        exit(1);
    }
    std::stringstream ss;
    ss << f.rdbuf();
    return ss.str();
}

int main(int argc, char **argv) {
    if (argc < 4) {
        fprintf(stderr, "usage: %s <skeletons dir> <log2n> <reps> [trace.bin|-] [nvrtc options]\n", argv[0]);
        return 1;
    }
    const std::string dir = argv[1];
    const int lg = atoi(argv[2]);
    const int reps = atoi(argv[3]);
    const char *trace_path = argc > 4 && strcmp(argv[4], "-") ? argv[4] : nullptr;
    std::vector<std::string> opts = {"--gpu-architecture=sm_100a", "-default-device", "-std=c++17", "-lineinfo",
                                     "--fmad=false"};
    for (int i = 5; i < argc; ++i) opts.push_back(argv[i]);
    if (trace_path) opts.push_back("-DSKEL_SCAN_TRACE");
    const std::string text = slurp(dir + "/prelude.cuh") +
                             "\nunsigned lab_add(unsigned x, unsigned y) { return x + y; }\n#define SKEL_FN ::lab_add\n" +
                             slurp(dir + "/red.cuh");
    nvrtcProgram prog;
    if (nvrtcCreateProgram(&prog, text.c_str(), "scan_lab.cu", 0, nullptr, nullptr) != NVRTC_SUCCESS) return 1;
    std::vector<const char *> copts;
    for (auto &o : opts) copts.push_back(o.c_str());
    const nvrtcResult cr = nvrtcCompileProgram(prog, (int)copts.size(), copts.data());
    if (cr != NVRTC_SUCCESS) {
        size_t ls = 0;
        nvrtcGetProgramLogSize(prog, &ls);
        std::string log(ls, '\0');
        nvrtcGetProgramLog(prog, &log[0]);
        fprintf(stderr, "%s\n", log.c_str());
        return 1;
    }
    size_t cs = 0;
    nvrtcGetCUBINSize(prog, &cs);
    std::vector<char> cubin(cs);
    nvrtcGetCUBIN(prog, cubin.data());

    CKR(cudaFree(nullptr));  // primary context
    CUmodule mod;
    CKD(cuModuleLoadData(&mod, cubin.data()));
    CUfunction k;
    CKD(cuModuleGetFunction(&k, mod, "skel_scan_kernel"));
    CUdeviceptr sig_p;
    size_t sig_b = 0;
    CKD(cuModuleGetGlobal(&sig_p, &sig_b, mod, "skel_sig"));
    std::vector<skel_u64> sig(sig_b / 8);
    CKD(cuMemcpyDtoH(sig.data(), sig_p, sig_b));
    const int threads = (int)sig[14];
    const size_t dsm = (size_t)sig[12];
    const skel_u64 SRB = sig[15] & 0xffff, CH = (sig[15] >> 16) & 0xffff, K = sig[8], STILE = SRB * K;
    const skel_u64 REPL = std::max<skel_u64>(1, (sig[15] >> 32) & 0xff);

    const skel_u64 n = 1ull << lg;
    int sms = 0;
    CKR(cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0));
    CKD(cuFuncSetAttribute(k, CU_FUNC_ATTRIBUTE_MAX_DYNAMIC_SHARED_SIZE_BYTES, (int)dsm));
    int occ = 0;
    CKD(cuOccupancyMaxActiveBlocksPerMultiprocessor(&occ, k, threads, dsm));
    const skel_u64 G = (skel_u64)sms * (skel_u64)std::max(occ, 1);
    unsigned *in = nullptr, *out = nullptr;
    CKR(cudaMalloc(&in, n * 4));
    CKR(cudaMalloc(&out, n * 4));
    lab_fill<<<sms * 8, 256>>>(in, n);
    const skel_u64 nft = n / STILE, per_slice = G * CH, nslices = (nft + per_slice - 1) / per_slice;
    const skel_u64 nstat = REPL * (std::max<skel_u64>(1, nslices) * G + 64);
    skel_u64 *status = nullptr;
    unsigned *counters = nullptr;
    unsigned long long *bad = nullptr;
    CKR(cudaMalloc(&status, nstat * 8));
    CKR(cudaMemset(status, 0, nstat * 8));
    CKR(cudaMalloc(&counters, 256));
    CKR(cudaMemset(counters, 0, 256));
    const unsigned one = 1;
    CKR(cudaMemcpy(counters + 3, &one, 4, cudaMemcpyHostToDevice));
    CKR(cudaMalloc(&bad, 8));
    CUtensorMap tin, tout;
    const skel_u64 rows = nft * SRB;
    int use_tma = make_map(&tin, in, rows, (unsigned)SRB / 2) && make_map(&tout, out, rows, (unsigned)SRB / 2);
    alignas(16) unsigned char identity[16] = {0}, args[64] = {0};
    const void *seed = nullptr, *cin = in;
    void *flags = nullptr, *aggv = nullptr, *incv = nullptr, *total = nullptr, *vout = out, *vstatus = status;
    void *vcounters = counters;
    unsigned *epoch_ptr = counters + 3;
    skel_u64 nn = n;
    void *params[] = {&tin, &tout, &cin, &vout, &nn, &use_tma, identity, &seed, &vstatus, &flags,
                      &aggv, &incv, &vcounters, &epoch_ptr, &total, args};
    cudaEvent_t e0, e1;
    CKR(cudaEventCreate(&e0));
    CKR(cudaEventCreate(&e1));
    std::vector<float> ms;
    for (int r = 0; r < reps + 3; ++r) {
        CKR(cudaEventRecord(e0));
        CKD(cuLaunchKernel(k, (unsigned)G, 1, 1, threads, 1, 1, use_tma ? (unsigned)dsm : 0, 0, params, nullptr));
        CKR(cudaEventRecord(e1));
        CKR(cudaEventSynchronize(e1));
        float t = 0;
        CKR(cudaEventElapsedTime(&t, e0, e1));
        if (r >= 3) ms.push_back(t);
    }
    CKR(cudaGetLastError());
    CKR(cudaMemset(bad, 0, 8));
    lab_check<<<sms * 8, 256>>>(in, out, n, bad);
    unsigned long long nbad = 0;
    CKR(cudaMemcpy(&nbad, bad, 8, cudaMemcpyDeviceToHost));
    std::sort(ms.begin(), ms.end());
    const double med = ms[ms.size() / 2];
    std::string os;
    for (size_t i = 5; i < opts.size(); ++i) os += opts[i] + " ";
    printf("{\"opts\": \"%s\", \"log2n\": %d, \"G\": %llu, \"threads\": %d, \"smem\": %zu, \"tile\": %llu, \"ch\": %llu, "
           "\"slices\": %llu, \"ms_med\": %.4f, \"ms_min\": %.4f, \"GBps\": %.1f, \"bad\": %llu, \"tma\": %d}\n",
           os.c_str(), lg, (unsigned long long)G, threads, dsm, STILE, CH, (unsigned long long)nslices, med, ms[0],
           8.0 * n / med / 1e6, nbad, use_tma);
    if (trace_path) {
        CUdeviceptr tp;
        size_t tb = 0;
        CKD(cuModuleGetGlobal(&tp, &tb, mod, "skel_scan_trace"));
        std::vector<skel_u64> tr(tb / 8);
        CKD(cuMemcpyDtoH(tr.data(), tp, tb));
        FILE *f = fopen(trace_path, "wb");
        const skel_u64 hdr[4] = {G, nslices, 1024, 148};  // then [6][1024][148] stamps
        fwrite(hdr, 8, 4, f);
        fwrite(tr.data(), 8, tr.size(), f);
        fclose(f);
    }
    return nbad ? 2 : 0;
}
