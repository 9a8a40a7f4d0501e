// internal.h -- private declarations of libskel (not part of the C-ABI).
#pragma once

#include <cuda_runtime.h>
#include <nccl.h>

#include <cstddef>
#include <cstdint>
#include <map>
#include <memory>
#include <set>
#include <string>
#include <unordered_map>
#include <vector>

#include "skel.h"

namespace skelrt {

// ---------------------------------------------------------------------------
// errors: every CUDA/NCCL/NVRTC failure becomes a status + message
// ---------------------------------------------------------------------------
struct Error {
    int status;
    std::string msg;
};

// ---------------------------------------------------------------------------
// JIT modules (NVRTC injection + kernel cache)
// ---------------------------------------------------------------------------
enum class Kind { Map = 0, Zip = 1, Red = 2, Idx = 3, Lanes = 4 };

struct Module {
    Kind kind;
    std::string key;
    cudaLibrary_t lib = nullptr;
    cudaKernel_t k_main = nullptr;  // skel_ew_kernel | skel_reduce_kernel
    cudaKernel_t k_main_u1 = nullptr;  // Map/Zip: one chunk in flight per thread (fewer registers)
    cudaKernel_t k_scan = nullptr;
    cudaKernel_t k_fold = nullptr;
    cudaKernel_t k_seed = nullptr;
    cudaKernel_t k_scan_agg = nullptr;    // small-vector Scan: tile aggregates
    cudaKernel_t k_scan_small = nullptr;  // small-vector Scan: seeded tile scans
    cudaKernel_t k_fold_aggs = nullptr;   // small-vector Reduce: ordered fold of the tile aggregates
    cudaKernel_t k_red_agg2 = nullptr;    // small-vector Reduce: aggregates of double-size tiles
    cudaKernel_t k_zipcomb = nullptr;  // Zip modules: fused combine + zip + broadcast (peer memory)
    cudaKernel_t k_zipcomb_mm = nullptr;  // ... the same through NVSwitch multicast (multimem)
    uint64_t sig[16 + 4 * 32] = {0};
    std::set<int> attr_set_on;  // devices on which smem attributes were set
    // element-wise grid policy (runtime.cpp ew_decide): 0 = UNROLL chunks in
    // flight per thread, 1 = one chunk per thread, 2 = one element per thread
    // through the scalar path, 3 = one chunk per thread with the low-register
    // kernel (k_main_u1), 4 = the scalar path through k_main_u1; decided on a
    // sample at the first launch of each size class
    static constexpr int kPolicies = 6;
    // (size class = log2 of the chunk count, hash of the scalar arguments) -> decided policy
    std::map<std::pair<int, uint64_t>, int> ew_policy;
    // decisions persist next to the cached cubin (<key>.policy, one line per
    // decision: device tag, size class, argument hash, policy), so a later
    // process -- or one under a profiler, where trial timings are meaningless --
    // launches what an earlier one measured; empty: no disk cache
    std::string policy_path;
    bool policy_loaded = false;
    int red_occ = 0;  // resident Reduce CTAs per SM (0 = not yet queried)
};

// signature accessors (layout documented in map.cuh / red.cuh)
struct ArgSlot {
    uint64_t size, align, isptr, off;
};

// ---------------------------------------------------------------------------
// devices
// ---------------------------------------------------------------------------
struct Slot {
    int d = 0;      // logical device index (0..D-1)
    int dev = 0;    // CUDA device ordinal
    int sms = 148;  // multiprocessor count
    int cc = 100;   // compute capability, major * 10 + minor
    cudaStream_t stream = nullptr;
    cudaEvent_t ev = nullptr;  // join event
    cudaEvent_t ev_scan = nullptr;  // after this slot's persistent Scan (chains slots sharing a GPU)
    // asynchronous downloads (skel_vector_download_part_async) run on their own
    // stream, so a D2H overlaps the next uploads and kernels of the main stream
    cudaStream_t dl_stream = nullptr;
    cudaEvent_t dl_ready = nullptr;  // main-stream point a download waits for
    bool ev_scan_live = false;      // ev_scan has been recorded at least once
    // grow-only workspace for reduce/scan partials, look-back status, seeds
    char *ws = nullptr;
    size_t ws_cap = 0;
    unsigned *counters = nullptr;  // [1] scan done, [2] reduce done, [3] scan epoch (device-resident)
    // look-back status words (only ever hold status words; zeroed at allocation)
    unsigned long long *st64 = nullptr;
    size_t st64_cap = 0;  // entries
    unsigned *fl32 = nullptr;
    size_t fl32_cap = 0;  // entries
    // scratch for rank-mode downloads
    char *scratch = nullptr;
    size_t scratch_cap = 0;
};

struct VmmRec {  // a VMM (cuMemCreate) allocation backing a vector buffer
    unsigned long long handle = 0;
    size_t size = 0;
    int dev = 0;
};

// a multicast object (NVSwitch NVLS) bound to every device's buffer of a vector
struct McRec {
    unsigned long long handle = 0;  // CUmemGenericAllocationHandle of the multicast object
    unsigned long long va = 0;      // its mapping (one address reaches all bound buffers)
    size_t size = 0;
    std::vector<char *> bases;      // the buffers it is bound to (one per local slot)
    std::vector<int> devs;
};

// rank mode: an NCCL symmetric window over a vector buffer (ncclMemAlloc +
// ncclCommWindowRegister(NCCL_WIN_COLL_SYMMETRIC)) and the pointers it gives
struct WinRec {
    ncclWindow_t win = nullptr;
    size_t size = 0;
    std::vector<char *> peers;  // every rank's buffer, load/store-accessible from here
    char *mc = nullptr;         // its multicast address (NVLS), if the device communicator has one
};

struct Buf {  // one logical device's storage of a vector
    char *base = nullptr;
    size_t cap = 0;    // bytes allocated at base
    size_t off = 0;    // element offset of the live data inside base
    size_t count = 0;  // live elements
    char *ptr(size_t es) const { return base ? base + off * es : nullptr; }
    // an asynchronous download still reading this buffer: writers wait for it
    cudaEvent_t dl_done = nullptr;
    bool dl_pending = false;
    // rank mode: every rank's `base` of this vector, opened through CUDA IPC
    std::vector<char *> peers;
    char *peers_of = nullptr;  // the local base the peer table was built for
};

}  // namespace skelrt

struct skel_vec_s;

struct skel_ctx_s {
    int D = 1;                   // logical devices
    bool rank_mode = false;      // one process per GPU, NCCL exchanges
    int rank = 0;                // rank mode: this process's logical device
    std::vector<skelrt::Slot> slots;  // local logical devices
    ncclComm_t comm = nullptr;
    int block_size = 0;
    std::string cache_dir;
    bool disk_cache = true;
    bool fmad = false;
    // every pair of distinct physical devices has peer access enabled (in-process
    // mode); the fused peer-memory paths need it, else they take the unfused one
    bool peer_all = true;
    bool peer_atomics = true;  // every distinct pair has native P2P atomics (the cross-device Reduce ticket)
    // vector buffers of at least vmm_min bytes are VMM allocations (cuMemCreate,
    // exportable), so one allocation can be bound to a multicast object; rank
    // mode keeps cudaMalloc (its fused tail opens peers through CUDA IPC)
    bool vmm_on = true;
    size_t vmm_min = 2u << 20;
    std::unordered_map<char *, skelrt::VmmRec> vmm;
    int mc_ok = -1;  // every local device supports multicast (-1: not yet queried)
    // rank mode, SKEL_NCCL_WINDOWS=1: the fused tail's vectors live in NCCL
    // symmetric windows (peer pointers and the NVLS multicast address come from
    // NCCL instead of CUDA IPC)
    bool nccl_windows = false;
    std::set<char *> nccl_mem;                        // buffers from ncclMemAlloc
    std::unordered_map<char *, skelrt::WinRec> wins;  // registered windows by buffer
    int devcomm_state = -1;                           // -1 not tried, 0 failed, 1 created
    void *devcomm = nullptr;                          // ncclDevComm (nccl_device/impl/comm__types.h)
    skel_stats stats{};
    std::string last_error;
    std::map<std::string, std::unique_ptr<skelrt::Module>> modules;
    std::unordered_map<std::string, skelrt::Module *> fast_modules;  // (kind, options, user text) -> module
    std::set<skel_vec_s *> vecs;
    bool capturing = false;  // between skel_capture_begin and skel_capture_end
    std::vector<std::pair<skel_vec_s *, uint64_t>> captured;  // vectors written inside the capture
    uint64_t next_serial = 0;
};

struct skel_graph_s {
    skel_ctx_s *ctx = nullptr;
    cudaGraph_t graph = nullptr;
    cudaGraphExec_t exec = nullptr;
    std::vector<std::pair<skel_vec_s *, uint64_t>> written;  // (vector, serial) the graph writes
};

struct skel_vec_s {
    skel_ctx_s *ctx = nullptr;
    size_t n = 0, es = 0;
    skel_dist dist = SKEL_SINGLE;
    skel_dtype dt = SKEL_DT_OPAQUE;
    char *host = nullptr;   // pinned mirror (lazily allocated)
    size_t host_lo = 0;     // mirror covers elements [host_lo, host_lo + host_n)
    size_t host_n = 0;      // == n except for a rank-local part mirror (upload_part)
    bool host_valid = false;
    bool dev_valid = true;  // created zero-filled on the devices
    bool diverged = false;  // copy distribution after mark_device_modified
    std::vector<skelrt::Buf> bufs;  // indexed like ctx->slots
    uint64_t serial = 0;            // unique per context (graphs refer to vectors by it)
    skelrt::McRec mc;               // multicast binding of bufs (fused NVLS tail), if any
};

namespace skelrt {
// jit.cpp
int get_module(skel_ctx_s *ctx, Kind kind, const char *src, Module **out);
std::string entry_name(const std::string &src, std::string *err);
// NVRTC compile without any device (used by skel_compile_check)
int compile_only(Kind kind, const char *src, int block, bool fmad, std::string *log, std::vector<char> *cubin);

// builtin.cu (nvcc-compiled helper kernels)
cudaError_t launch_fill(void *dst, size_t n, const void *elem, size_t es, cudaStream_t s);
// dst[i] = op(srcs[0][i], ..., srcs[nsrc-1][i]) for i < count; dst may alias srcs[j]
cudaError_t launch_combine(void *dst, const void *const *srcs, int nsrc, size_t count, skel_dtype dt,
                           skel_combine op, cudaStream_t s);
// dst[j*bytes ...] = srcs[j][0 .. bytes) for j < nsrc
cudaError_t launch_gather(void *dst, const void *const *srcs, int nsrc, size_t bytes, cudaStream_t s);
}  // namespace skelrt
