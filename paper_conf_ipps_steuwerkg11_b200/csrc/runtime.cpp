// runtime.cpp -- the host side of libskel: contexts, the Vector coherence
// tracker, the distribution planner/executor and the skeleton launchers,
// exported through the C-ABI of include/skel.h.
//
// Paper passages implemented here:
//  * Vector + lazy coherence (§III-A): a vector has a (pinned)
//    host mirror and per-device storage; each side carries a valid bit; a
//    transfer happens only when the destination is stale;
//    skeleton outputs stay on the devices.
//  * Distributions (§III-D; Listing 4): single /
//    block / copy placement over D logical devices, redistribution with data
//    exchange, copy -> block with element-wise combine.
//  * Skeleton execution on several devices: block parts run on
//    their own device; Reduce/Scan add one exchange of D partial results and an
//    ordered fold (cross-device combination in device order).
#include <cuda.h>
#include <cudaTypedefs.h>

#include <algorithm>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <fcntl.h>
#include <fstream>
#include <unistd.h>
#include <mutex>

#include <nccl_device/impl/comm__types.h>  // host views of ncclDevComm / ncclWindow_vidmem
#include <nvtx3/nvToolsExt.h>

#include "internal.h"

using namespace skelrt;

// NVTX ranges: every skeleton call and every planner operation
// is a named range in the "skel" domain, so Nsight timelines show the paper's
// operations (Map/Zip/Reduce/Scan, distribution changes, transfers) around the
// kernels and collectives they launch.  Header-only NVTX3: free unless a tool
// is attached.
namespace {
nvtxDomainHandle_t nvtx_domain() {
    static nvtxDomainHandle_t d = nvtxDomainCreateA("skel");
    return d;
}
struct NvtxRange {
    explicit NvtxRange(const char *name) {
        nvtxEventAttributes_t a = {};
        a.version = NVTX_VERSION;
        a.size = NVTX_EVENT_ATTRIB_STRUCT_SIZE;
        a.messageType = NVTX_MESSAGE_TYPE_ASCII;
        a.message.ascii = name;
        nvtxDomainRangePushEx(nvtx_domain(), &a);
    }
    ~NvtxRange() { nvtxDomainRangePop(nvtx_domain()); }
};
}  // namespace
#define SKEL_RANGE(name) NvtxRange skel_nvtx_range_(name)

namespace {

thread_local std::string g_last_error;  // failures without a context

int fail(skel_ctx_s *ctx, int st, const std::string &msg) {
    if (ctx) ctx->last_error = msg;
    else g_last_error = msg;
    if (getenv("SKEL_LOG")) fprintf(stderr, "[skel] error %d: %s\n", st, msg.c_str());
    return st;
}

#define CK(ctx, call)                                                                                      \
    do {                                                                                                   \
        cudaError_t _e = (call);                                                                           \
        if (_e != cudaSuccess)                                                                             \
            return fail((ctx), SKEL_ERR_CUDA, std::string(#call) + ": " + cudaGetErrorString(_e));         \
    } while (0)
#define NK(ctx, call)                                                                                      \
    do {                                                                                                   \
        ncclResult_t _r = (call);                                                                          \
        if (_r != ncclSuccess)                                                                             \
            return fail((ctx), SKEL_ERR_NCCL, std::string(#call) + ": " + ncclGetErrorString(_r));         \
    } while (0)
#define TRY(expr)                          \
    do {                                   \
        int _s = (expr);                   \
        if (_s != SKEL_OK) return _s;      \
    } while (0)

inline size_t part_size(size_t n, int D) { return D > 0 ? (n + D - 1) / D : 0; }
inline void part_range(size_t n, int D, int k, size_t *lo, size_t *hi) {
    const size_t s = part_size(n, D);
    *lo = std::min(n, (size_t)k * s);
    *hi = std::min(n, (size_t)(k + 1) * s);
}
inline size_t align_up(size_t x, size_t a) { return (x + a - 1) / a * a; }
inline bool al16(const void *p) { return (reinterpret_cast<uintptr_t>(p) & 15) == 0; }

size_t want_count(const skel_vec_s *v, skel_dist dist, int d) {
    size_t lo, hi;
    switch (dist) {
        case SKEL_SINGLE: return d == 0 ? v->n : 0;
        case SKEL_COPY: return v->n;
        default: part_range(v->n, v->ctx->D, d, &lo, &hi); return hi - lo;
    }
}
size_t part_lo(const skel_vec_s *v, int d) {
    size_t lo, hi;
    part_range(v->n, v->ctx->D, d, &lo, &hi);
    return lo;
}
// bytes of a "full" per-device buffer: D parts of ceil(n/D) elements (NCCL
// collectives need equal part sizes; the padding is never read as data)
size_t full_bytes(const skel_vec_s *v) {
    return std::max<size_t>(part_size(v->n, v->ctx->D) * v->ctx->D * v->es, 16);
}

struct DevGuard {
    explicit DevGuard(int dev) { cudaSetDevice(dev); }
};

int wait_dl(skel_vec_s *v);
int sync_downloads(skel_ctx_s *ctx);

// ---- CUDA driver entry points (VMM, multicast), resolved through the runtime ----
struct Drv {
    PFN_cuMemCreate_v10020 create = nullptr;
    PFN_cuMemRelease_v10020 release = nullptr;
    PFN_cuMemAddressReserve_v10020 reserve = nullptr;
    PFN_cuMemAddressFree_v10020 addr_free = nullptr;
    PFN_cuMemMap_v10020 map = nullptr;
    PFN_cuMemUnmap_v10020 unmap = nullptr;
    PFN_cuMemSetAccess_v10020 set_access = nullptr;
    PFN_cuMemGetAllocationGranularity_v10020 granularity = nullptr;
    PFN_cuMulticastCreate_v12010 mc_create = nullptr;
    PFN_cuMulticastAddDevice_v12010 mc_add = nullptr;
    PFN_cuMulticastBindMem_v12010 mc_bind = nullptr;
    PFN_cuMulticastUnbind_v12010 mc_unbind = nullptr;
    PFN_cuMulticastGetGranularity_v12010 mc_granularity = nullptr;
    PFN_cuDeviceGetAttribute_v2000 attr = nullptr;
    bool vmm = false, mc = false;
};
const Drv &drv() {
    static Drv d;
    static std::once_flag once;
    std::call_once(once, [] {
        auto get = [](const char *name, int ver, void **fn) {
            cudaDriverEntryPointQueryResult q;
            if (cudaGetDriverEntryPointByVersion(name, fn, ver, cudaEnableDefault, &q) != cudaSuccess ||
                q != cudaDriverEntryPointSuccess) {
                cudaGetLastError();
                *fn = nullptr;
            }
        };
        get("cuMemCreate", 10020, (void **)&d.create);
        get("cuMemRelease", 10020, (void **)&d.release);
        get("cuMemAddressReserve", 10020, (void **)&d.reserve);
        get("cuMemAddressFree", 10020, (void **)&d.addr_free);
        get("cuMemMap", 10020, (void **)&d.map);
        get("cuMemUnmap", 10020, (void **)&d.unmap);
        get("cuMemSetAccess", 10020, (void **)&d.set_access);
        get("cuMemGetAllocationGranularity", 10020, (void **)&d.granularity);
        get("cuMulticastCreate", 12010, (void **)&d.mc_create);
        get("cuMulticastAddDevice", 12010, (void **)&d.mc_add);
        get("cuMulticastBindMem", 12010, (void **)&d.mc_bind);
        get("cuMulticastUnbind", 12010, (void **)&d.mc_unbind);
        get("cuMulticastGetGranularity", 12010, (void **)&d.mc_granularity);
        get("cuDeviceGetAttribute", 2000, (void **)&d.attr);
        d.vmm = d.create && d.release && d.reserve && d.addr_free && d.map && d.unmap && d.set_access &&
                d.granularity;
        d.mc = d.vmm && d.mc_create && d.mc_add && d.mc_bind && d.mc_unbind && d.mc_granularity && d.attr;
    });
    return d;
}

// distinct physical devices of the context's local slots
std::vector<int> local_devices(const skel_ctx_s *ctx) {
    std::vector<int> devs;
    for (const auto &s : ctx->slots)
        if (std::find(devs.begin(), devs.end(), s.dev) == devs.end()) devs.push_back(s.dev);
    return devs;
}

// ---- device memory -----------------------------------------------------------
// VMM allocation (cuMemCreate + cuMemMap) on slot s's device, readable and
// writable from every local device (in-process peers need cuMemSetAccess, not
// cudaDeviceEnablePeerAccess, for VMM memory).  The physical memory is
// exportable as a POSIX file descriptor where the driver allows it.  Size:
// rounded up to the allocation granularity (2 MB), which is also the minimum
// multicast granularity, so the buffer can be bound to a multicast object.
// *out = nullptr (and SKEL_OK) when VMM is unavailable: the caller falls back.
int vmm_alloc(skel_ctx_s *ctx, Slot &s, size_t bytes, char **out) {
    *out = nullptr;
    const Drv &d = drv();
    if (!d.vmm) return SKEL_OK;
    DevGuard g(s.dev);
    CUmemAllocationProp prop = {};
    prop.type = CU_MEM_ALLOCATION_TYPE_PINNED;
    prop.location.type = CU_MEM_LOCATION_TYPE_DEVICE;
    prop.location.id = s.dev;
    prop.requestedHandleTypes = CU_MEM_HANDLE_TYPE_POSIX_FILE_DESCRIPTOR;
    size_t gran = 0;
    if (d.granularity(&gran, &prop, CU_MEM_ALLOC_GRANULARITY_RECOMMENDED) != CUDA_SUCCESS || !gran) return SKEL_OK;
    const size_t size = align_up(std::max<size_t>(bytes, 1), gran);
    CUmemGenericAllocationHandle h = 0;
    CUresult r = d.create(&h, size, &prop, 0);
    if (r != CUDA_SUCCESS) {  // not exportable here: a plain VMM allocation
        prop.requestedHandleTypes = CU_MEM_HANDLE_TYPE_NONE;
        r = d.create(&h, size, &prop, 0);
    }
    if (r == CUDA_ERROR_OUT_OF_MEMORY) return fail(ctx, SKEL_ERR_OOM, "cuMemCreate(" + std::to_string(size) + ")");
    if (r != CUDA_SUCCESS) return SKEL_OK;
    CUdeviceptr va = 0;
    if (d.reserve(&va, size, gran, 0, 0) != CUDA_SUCCESS) {
        d.release(h);
        return SKEL_OK;
    }
    std::vector<CUmemAccessDesc> acc;
    for (int dev : local_devices(ctx)) {
        CUmemAccessDesc a = {};
        a.location.type = CU_MEM_LOCATION_TYPE_DEVICE;
        a.location.id = dev;
        a.flags = CU_MEM_ACCESS_FLAGS_PROT_READWRITE;
        acc.push_back(a);
    }
    if (d.map(va, size, 0, h, 0) != CUDA_SUCCESS || d.set_access(va, size, acc.data(), acc.size()) != CUDA_SUCCESS) {
        d.unmap(va, size);
        d.addr_free(va, size);
        d.release(h);
        return SKEL_OK;
    }
    char *p = reinterpret_cast<char *>(va);
    ctx->vmm[p] = VmmRec{(unsigned long long)h, size, s.dev};
    ctx->stats.vmm_allocs++;
    *out = p;
    return SKEL_OK;
}

int dev_alloc(skel_ctx_s *ctx, Slot &s, size_t bytes, char **out) {
    DevGuard g(s.dev);
    void *p = nullptr;
    cudaError_t e = cudaMalloc(&p, std::max<size_t>(bytes, 256));
    if (e != cudaSuccess) {
        cudaGetLastError();
        return fail(ctx, SKEL_ERR_OOM, std::string("cudaMalloc(") + std::to_string(bytes) + "): " +
                                           cudaGetErrorString(e));
    }
    *out = static_cast<char *>(p);
    return SKEL_OK;
}
int dev_free(skel_ctx_s *ctx, Slot &s, char *p) {
    if (!p) return SKEL_OK;
    if (ctx->capturing)
        return fail(ctx, SKEL_ERR_STATE, "a buffer would be reallocated inside a capture: run the sequence once "
                                         "eagerly before capturing it");
    DevGuard g(s.dev);
    CK(ctx, cudaStreamSynchronize(s.stream));
    if (s.dl_stream) CK(ctx, cudaStreamSynchronize(s.dl_stream));  // a download may still read it
    if (ctx->nccl_mem.count(p)) {  // rank mode: an NCCL symmetric window's buffer
        auto w = ctx->wins.find(p);
        if (w != ctx->wins.end()) {
            ncclCommWindowDeregister(ctx->comm, w->second.win);  // collective, like the registration
            ctx->wins.erase(w);
        }
        ncclMemFree(p);
        ctx->nccl_mem.erase(p);
        return SKEL_OK;
    }
    auto it = ctx->vmm.find(p);
    if (it != ctx->vmm.end()) {
        const Drv &d = drv();
        for (auto &o : ctx->slots)  // peers may still read it (exchanges): drain every local stream
            if (&o != &s) {
                DevGuard go(o.dev);
                cudaStreamSynchronize(o.stream);
            }
        const CUdeviceptr va = reinterpret_cast<CUdeviceptr>(p);
        d.unmap(va, it->second.size);
        d.addr_free(va, it->second.size);
        d.release((CUmemGenericAllocationHandle)it->second.handle);
        ctx->vmm.erase(it);
        return SKEL_OK;
    }
    CK(ctx, cudaFree(p));
    return SKEL_OK;
}

// storage of a vector buffer: VMM when large enough (in-process contexts)
int vec_alloc(skel_ctx_s *ctx, Slot &s, size_t bytes, char **out) {
    if (!ctx->rank_mode && ctx->vmm_on && bytes >= ctx->vmm_min) {
        TRY(vmm_alloc(ctx, s, bytes, out));
        if (*out) return SKEL_OK;
    }
    return dev_alloc(ctx, s, bytes, out);
}

// ---- multicast (NVLS) binding of a vector's device buffers -----------------------
void mc_release(skel_vec_s *v) {
    McRec &m = v->mc;
    if (!m.handle) return;
    const Drv &d = drv();
    skel_ctx_s *ctx = v->ctx;
    for (auto &s : ctx->slots) {
        DevGuard g(s.dev);
        cudaStreamSynchronize(s.stream);
    }
    d.unmap((CUdeviceptr)m.va, m.size);
    d.addr_free((CUdeviceptr)m.va, m.size);
    for (int dev : m.devs) d.mc_unbind((CUmemGenericAllocationHandle)m.handle, (CUdevice)dev, 0, m.size);
    d.release((CUmemGenericAllocationHandle)m.handle);
    m = McRec{};
}
// release the multicast binding of any vector bound to buffer p (before p is freed)
void mc_release_base(skel_ctx_s *ctx, const char *p) {
    for (skel_vec_s *v : ctx->vecs)
        if (v->mc.handle && std::find(v->mc.bases.begin(), v->mc.bases.end(), p) != v->mc.bases.end())
            mc_release(v);
}

// every local device supports multicast (queried once)
bool mc_supported(skel_ctx_s *ctx) {
    if (ctx->mc_ok >= 0) return ctx->mc_ok == 1;
    const Drv &d = drv();
    bool ok = d.mc && !ctx->rank_mode;
    if (const char *e = getenv("SKEL_MULTIMEM")) ok = ok && atoi(e) != 0;
    for (int dev : local_devices(ctx)) {
        int v = 0;
        CUresult r = ok ? d.attr(&v, CU_DEVICE_ATTRIBUTE_MULTICAST_SUPPORTED, (CUdevice)dev) : CUDA_SUCCESS;
        if (getenv("SKEL_LOG"))
            fprintf(stderr, "[skel] multicast: driver entry points %d, device %d attribute %d (query %d)\n", (int)d.mc,
                    dev, v, (int)r);
        if (!ok || r != CUDA_SUCCESS || !v) ok = false;
    }
    ctx->mc_ok = ok ? 1 : 0;
    return ok;
}

// one multicast object bound to the first `bytes` of every local slot's buffer
// of v (each slot a distinct device, every buffer a VMM allocation large
// enough); false (no error) if that is not possible
bool mc_bind(skel_vec_s *v, size_t bytes) {
    skel_ctx_s *ctx = v->ctx;
    std::vector<char *> bases;
    for (auto &b : v->bufs) bases.push_back(b.base);
    if (v->mc.handle && v->mc.bases == bases && v->mc.size >= bytes) return true;
    mc_release(v);
    if (!mc_supported(ctx) || local_devices(ctx).size() != ctx->slots.size()) return false;
    const Drv &d = drv();
    CUmulticastObjectProp prop = {};
    prop.numDevices = (unsigned)ctx->slots.size();
    prop.handleTypes = CU_MEM_HANDLE_TYPE_NONE;
    prop.size = std::max<size_t>(bytes, 1);
    size_t gran = 0;
    if (d.mc_granularity(&gran, &prop, CU_MULTICAST_GRANULARITY_MINIMUM) != CUDA_SUCCESS || !gran) return false;
    prop.size = align_up(prop.size, gran);
    for (auto &b : v->bufs) {
        auto it = ctx->vmm.find(b.base);
        if (it == ctx->vmm.end() || it->second.size < prop.size) return false;
    }
    CUmemGenericAllocationHandle mc = 0;
    // the handle type of the multicast object: exportable kinds first (what the
    // driver accepts depends on the platform), then none
    CUresult cr = CUDA_ERROR_INVALID_VALUE;
    for (CUmemAllocationHandleType ht : {CU_MEM_HANDLE_TYPE_POSIX_FILE_DESCRIPTOR, CU_MEM_HANDLE_TYPE_FABRIC,
                                         CU_MEM_HANDLE_TYPE_NONE}) {
        prop.handleTypes = ht;
        cr = d.mc_create(&mc, &prop);
        if (getenv("SKEL_LOG"))
            fprintf(stderr, "[skel] cuMulticastCreate(handle type %d, size %zu, devices %u): %d\n", (int)ht,
                    (size_t)prop.size, prop.numDevices, (int)cr);
        if (cr == CUDA_SUCCESS) break;
    }
    if (cr != CUDA_SUCCESS) {
        cudaGetLastError();
        return false;
    }
    McRec m;
    m.handle = (unsigned long long)mc;
    m.size = prop.size;
    bool ok = true;
    for (auto &s : ctx->slots) ok = ok && d.mc_add(mc, (CUdevice)s.dev) == CUDA_SUCCESS;
    for (size_t li = 0; ok && li < ctx->slots.size(); ++li) {
        DevGuard g(ctx->slots[li].dev);
        const VmmRec &r = ctx->vmm[v->bufs[li].base];
        ok = d.mc_bind(mc, 0, (CUmemGenericAllocationHandle)r.handle, 0, prop.size, 0) == CUDA_SUCCESS;
        if (ok) m.devs.push_back(ctx->slots[li].dev);
    }
    CUdeviceptr va = 0;
    if (ok) ok = d.reserve(&va, prop.size, gran, 0, 0) == CUDA_SUCCESS;
    if (ok) {
        ok = d.map(va, prop.size, 0, mc, 0) == CUDA_SUCCESS;
        std::vector<CUmemAccessDesc> acc;
        for (auto &s : ctx->slots) {
            CUmemAccessDesc a = {};
            a.location.type = CU_MEM_LOCATION_TYPE_DEVICE;
            a.location.id = s.dev;
            a.flags = CU_MEM_ACCESS_FLAGS_PROT_READWRITE;
            acc.push_back(a);
        }
        if (ok) ok = d.set_access(va, prop.size, acc.data(), acc.size()) == CUDA_SUCCESS;
        if (!ok) {
            d.unmap(va, prop.size);
            d.addr_free(va, prop.size);
        }
    }
    if (!ok) {
        if (getenv("SKEL_LOG")) fprintf(stderr, "[skel] multicast bind/map failed\n");
        cudaGetLastError();
        for (int dev : m.devs) d.mc_unbind(mc, (CUdevice)dev, 0, prop.size);
        d.release(mc);
        return false;
    }
    m.va = (unsigned long long)va;
    m.bases = bases;
    v->mc = m;
    ctx->stats.mc_binds++;
    return true;
}
// make b hold at least `bytes`; the first `keep` bytes at element offset
// b.off move to byte offset new_off_bytes of the new allocation
int buf_grow(skel_ctx_s *ctx, Slot &s, Buf &b, size_t bytes, size_t es, size_t keep, size_t new_off_elems) {
    if (b.cap >= bytes && (keep == 0 || b.off == new_off_elems)) {
        b.off = new_off_elems;
        return SKEL_OK;
    }
    if (b.cap >= bytes && keep) {  // same buffer, move data
        DevGuard g(s.dev);
        CK(ctx, cudaMemcpyAsync(b.base + new_off_elems * es, b.base + b.off * es, keep, cudaMemcpyDeviceToDevice,
                                s.stream));
        b.off = new_off_elems;
        return SKEL_OK;
    }
    char *nb = nullptr;
    TRY(vec_alloc(ctx, s, bytes, &nb));
    DevGuard g(s.dev);
    if (keep) CK(ctx, cudaMemcpyAsync(nb + new_off_elems * es, b.base + b.off * es, keep, cudaMemcpyDeviceToDevice,
                                      s.stream));
    if (b.base) mc_release_base(ctx, b.base);
    TRY(dev_free(ctx, s, b.base));
    b.base = nb;
    b.cap = bytes;
    b.off = new_off_elems;
    return SKEL_OK;
}

// Place the (uninitialised) storage of v for `dist` on every local device.
// Block parts sit at offset lo when the buffer is a full one (so that NCCL's
// in-place all-gather / reduce-scatter layout holds), else at 0.
int place(skel_vec_s *v, skel_dist dist) {
    skel_ctx_s *ctx = v->ctx;
    for (size_t li = 0; li < ctx->slots.size(); ++li) {
        Slot &s = ctx->slots[li];
        Buf &b = v->bufs[li];
        const size_t cnt = want_count(v, dist, s.d);
        size_t need, off = 0;
        if (dist == SKEL_COPY) {
            need = full_bytes(v);
        } else if (dist == SKEL_BLOCK) {
            const size_t fb = full_bytes(v);
            if (b.cap >= fb) {
                need = fb;
                off = part_lo(v, s.d);
            } else {
                need = std::max<size_t>(part_size(v->n, ctx->D) * v->es, 16);
            }
        } else {
            need = std::max<size_t>(cnt * v->es, 16);
        }
        if (b.cap < need) TRY(buf_grow(ctx, s, b, need, v->es, 0, 0));
        b.off = off;
        b.count = cnt;
    }
    return SKEL_OK;
}

// every local stream waits for all others (exchanges between logical devices)
int join(skel_ctx_s *ctx) {
    if (ctx->slots.size() < 2) return SKEL_OK;
    for (auto &s : ctx->slots) {
        DevGuard g(s.dev);
        CK(ctx, cudaEventRecord(s.ev, s.stream));
    }
    for (auto &s : ctx->slots) {
        DevGuard g(s.dev);
        for (auto &o : ctx->slots)
            if (&o != &s) CK(ctx, cudaStreamWaitEvent(s.stream, o.ev, 0));
    }
    return SKEL_OK;
}

bool partial_mirror(const skel_vec_s *v) { return v->host && v->host_n != v->n; }

// the devices now hold newer data than the host; inside a capture the vector
// is also remembered, so that replaying the graph invalidates its host copy
void device_wrote(skel_vec_s *v) {
    v->host_valid = false;
    if (v->ctx->capturing) v->ctx->captured.emplace_back(v, v->serial);
}

int host_mirror(skel_vec_s *v) {
    if (v->host && !partial_mirror(v)) return SKEL_OK;
    if (v->host) {  // a rank-local part mirror is replaced by a full one
        cudaFreeHost(v->host);
        v->host = nullptr;
    }
    v->host_lo = 0;
    v->host_n = v->n;
    void *p = nullptr;
    cudaError_t e = cudaHostAlloc(&p, std::max<size_t>(v->n * v->es, 16), cudaHostAllocPortable);
    if (e != cudaSuccess) {
        cudaGetLastError();
        return fail(v->ctx, SKEL_ERR_OOM, std::string("cudaHostAlloc: ") + cudaGetErrorString(e));
    }
    v->host = static_cast<char *>(p);
    return SKEL_OK;
}

// lazy H2D: make the devices hold v's data
int ensure_device(skel_vec_s *v) {
    if (v->dev_valid) return SKEL_OK;
    skel_ctx_s *ctx = v->ctx;
    if (!v->host_valid || !v->host) return fail(ctx, SKEL_ERR_STATE, "vector has no valid copy");
    TRY(wait_dl(v));
    TRY(place(v, v->dist));
    for (size_t li = 0; li < ctx->slots.size(); ++li) {
        Slot &s = ctx->slots[li];
        Buf &b = v->bufs[li];
        if (!b.count) continue;
        const size_t lo = (v->dist == SKEL_BLOCK) ? part_lo(v, s.d) : 0;
        if (lo < v->host_lo || lo + b.count > v->host_lo + v->host_n)
            return fail(ctx, SKEL_ERR_STATE, "host data of this part were not uploaded (upload_part covers another range)");
        DevGuard g(s.dev);
        CK(ctx, cudaMemcpyAsync(b.ptr(v->es), v->host + (lo - v->host_lo) * v->es, b.count * v->es,
                                cudaMemcpyHostToDevice, s.stream));
        ctx->stats.h2d_bytes += b.count * v->es;
        ctx->stats.h2d_copies++;
    }
    v->dev_valid = true;
    v->diverged = false;
    return SKEL_OK;
}

int sync_all(skel_ctx_s *ctx) {
    if (ctx->capturing) return fail(ctx, SKEL_ERR_STATE, "blocking call inside a capture (skel_capture_begin)");
    for (auto &s : ctx->slots) {
        DevGuard g(s.dev);
        CK(ctx, cudaStreamSynchronize(s.stream));
    }
    if (ctx->comm) {
        ncclResult_t ae = ncclSuccess;
        NK(ctx, ncclCommGetAsyncError(ctx->comm, &ae));
        if (ae != ncclSuccess) return fail(ctx, SKEL_ERR_NCCL, std::string("NCCL async: ") + ncclGetErrorString(ae));
    }
    return SKEL_OK;
}

// every asynchronous download has finished
int sync_downloads(skel_ctx_s *ctx) {
    for (auto &s : ctx->slots) {
        DevGuard g(s.dev);
        CK(ctx, cudaStreamSynchronize(s.dl_stream));
    }
    return SKEL_OK;
}

// v is about to be written on the main streams: wait (on the device) for any
// asynchronous download still reading its buffers
int wait_dl(skel_vec_s *v) {
    skel_ctx_s *ctx = v->ctx;
    for (size_t li = 0; li < v->bufs.size(); ++li) {
        Buf &b = v->bufs[li];
        if (!b.dl_pending) continue;
        Slot &s = ctx->slots[li];
        DevGuard g(s.dev);
        CK(ctx, cudaStreamWaitEvent(s.stream, b.dl_done, 0));
        b.dl_pending = false;
    }
    return SKEL_OK;
}

int scratch(skel_ctx_s *ctx, Slot &s, size_t bytes) {
    if (s.scratch_cap >= bytes) return SKEL_OK;
    TRY(dev_free(ctx, s, s.scratch));
    s.scratch = nullptr;
    s.scratch_cap = 0;
    TRY(dev_alloc(ctx, s, bytes, &s.scratch));
    s.scratch_cap = bytes;
    return SKEL_OK;
}

// lazy D2H into the host mirror
int ensure_host(skel_vec_s *v) {
    if (v->host_valid && !partial_mirror(v)) return SKEL_OK;
    if (partial_mirror(v)) {
        TRY(ensure_device(v));
        v->host_valid = false;
    }
    skel_ctx_s *ctx = v->ctx;
    TRY(host_mirror(v));
    const size_t es = v->es;
    if (!ctx->rank_mode) {
        for (size_t li = 0; li < ctx->slots.size(); ++li) {
            Slot &s = ctx->slots[li];
            Buf &b = v->bufs[li];
            if (!b.count) continue;
            if (v->dist == SKEL_COPY && s.d != 0) continue;  // read device 0's copy (reading R6)
            const size_t lo = (v->dist == SKEL_BLOCK) ? part_lo(v, s.d) : 0;
            DevGuard g(s.dev);
            CK(ctx, cudaMemcpyAsync(v->host + lo * es, b.ptr(es), b.count * es, cudaMemcpyDeviceToHost, s.stream));
            ctx->stats.d2h_bytes += b.count * es;
            ctx->stats.d2h_copies++;
        }
    } else {
        Slot &s = ctx->slots[0];
        Buf &b = v->bufs[0];
        DevGuard g(s.dev);
        const char *src = b.ptr(es);
        if (ctx->D > 1 && v->dist != SKEL_COPY) {
            const size_t ps = part_size(v->n, ctx->D);
            TRY(scratch(ctx, s, std::max<size_t>(ps * ctx->D * es, 16)));
            if (v->dist == SKEL_BLOCK) {
                NK(ctx, ncclAllGather(b.ptr(es), s.scratch, ps * es, ncclUint8, ctx->comm, s.stream));
            } else {  // SINGLE: rank 0 broadcasts
                NK(ctx, ncclBroadcast(s.d == 0 ? b.ptr(es) : s.scratch, s.scratch, v->n * es, ncclUint8, 0, ctx->comm,
                                      s.stream));
            }
            ctx->stats.nccl_bytes += ps * ctx->D * es;
            src = s.scratch;
        } else if (ctx->D > 1 && v->diverged) {
            TRY(scratch(ctx, s, std::max<size_t>(v->n * es, 16)));
            NK(ctx, ncclBroadcast(b.ptr(es), s.scratch, v->n * es, ncclUint8, 0, ctx->comm, s.stream));
            ctx->stats.nccl_bytes += v->n * es;
            src = s.scratch;
        }
        if (v->n) {
            CK(ctx, cudaMemcpyAsync(v->host, src, v->n * es, cudaMemcpyDeviceToHost, s.stream));
            ctx->stats.d2h_bytes += v->n * es;
            ctx->stats.d2h_copies++;
        }
    }
    TRY(sync_all(ctx));
    v->host_valid = true;
    return SKEL_OK;
}

ncclDataType_t nccl_type(skel_dtype dt) {
    switch (dt) {
        case SKEL_DT_F32: return ncclFloat32;
        case SKEL_DT_F64: return ncclFloat64;
        case SKEL_DT_I32: return ncclInt32;
        case SKEL_DT_U32: return ncclUint32;
        case SKEL_DT_I64: return ncclInt64;
        case SKEL_DT_U64: return ncclUint64;
        default: return ncclUint8;
    }
}
ncclRedOp_t nccl_op(skel_combine c) {
    switch (c) {
        case SKEL_COMBINE_MIN: return ncclMin;
        case SKEL_COMBINE_MAX: return ncclMax;
        case SKEL_COMBINE_PROD: return ncclProd;
        default: return ncclSum;
    }
}

int plan_exchange(skel_dist from, skel_dist to, skel_combine combine) {
    if (combine != SKEL_COMBINE_NONE) {
        if (from != SKEL_COPY) return -1;
        if (to == SKEL_BLOCK) return SKEL_XCHG_REDUCE_SCATTER;
        if (to == SKEL_SINGLE) return SKEL_XCHG_REDUCE;
        return SKEL_XCHG_ALLREDUCE;
    }
    if (from == to) return SKEL_XCHG_NONE;
    if (from == SKEL_SINGLE) return to == SKEL_BLOCK ? SKEL_XCHG_SCATTER : SKEL_XCHG_BROADCAST;
    if (from == SKEL_BLOCK) return to == SKEL_SINGLE ? SKEL_XCHG_GATHER : SKEL_XCHG_ALLGATHER;
    return to == SKEL_BLOCK ? SKEL_XCHG_LOCAL_SLICE : SKEL_XCHG_KEEP_ROOT;
}

// Kernels that read other devices' buffers (combine, gather) need peer access.
// Without it between some pair of GPUs (ctx->peer_all false), every operand on
// another physical device is first copied into slot s's scratch (cudaMemcpy
// stages through the host when P2P is unavailable) and read from there.
int stage_remote(skel_ctx_s *ctx, Slot &s, std::vector<const void *> &src, const std::vector<int> &src_dev,
                 size_t bytes) {
    if (ctx->peer_all) return SKEL_OK;
    size_t remote = 0;
    for (size_t j = 0; j < src.size(); ++j) remote += src_dev[j] != s.dev;
    if (!remote) return SKEL_OK;
    const size_t stride = align_up(std::max<size_t>(bytes, 1), 256);
    TRY(scratch(ctx, s, stride * remote));
    DevGuard g(s.dev);
    size_t k = 0;
    for (size_t j = 0; j < src.size(); ++j) {
        if (src_dev[j] == s.dev) continue;
        char *dst = s.scratch + stride * k++;
        if (bytes) CK(ctx, cudaMemcpyAsync(dst, src[j], bytes, cudaMemcpyDefault, s.stream));
        ctx->stats.d2d_bytes += bytes;
        src[j] = dst;
    }
    return SKEL_OK;
}

// ---- the exchanges (DESIGN.md §5 table T1) -----------------------------------
// Local mode: every logical device is in this process; data moves with
// cudaMemcpyAsync (peer or same GPU) and the combine kernel.
int xchg_local(skel_vec_s *v, int x, skel_combine combine) {
    skel_ctx_s *ctx = v->ctx;
    const int D = ctx->D;
    const size_t es = v->es, n = v->n;
    auto &S = ctx->slots;
    auto &B = v->bufs;
    TRY(join(ctx));
    switch (x) {
        case SKEL_XCHG_SCATTER: {
            for (int d = 1; d < D; ++d) {
                const size_t cnt = want_count(v, SKEL_BLOCK, d);
                if (B[d].cap < std::max<size_t>(part_size(n, D) * es, 16))
                    TRY(buf_grow(ctx, S[d], B[d], std::max<size_t>(part_size(n, D) * es, 16), es, 0, 0));
                B[d].off = 0;
                B[d].count = cnt;
                if (cnt) {
                    DevGuard g(S[d].dev);
                    CK(ctx, cudaMemcpyAsync(B[d].ptr(es), B[0].ptr(es) + part_lo(v, d) * es, cnt * es,
                                            cudaMemcpyDefault, S[d].stream));
                    ctx->stats.d2d_bytes += cnt * es;
                }
            }
            B[0].count = want_count(v, SKEL_BLOCK, 0);
            break;
        }
        case SKEL_XCHG_BROADCAST: {
            TRY(buf_grow(ctx, S[0], B[0], full_bytes(v), es, n * es, 0));
            for (int d = 1; d < D; ++d) {
                if (B[d].cap < full_bytes(v)) TRY(buf_grow(ctx, S[d], B[d], full_bytes(v), es, 0, 0));
                B[d].off = 0;
                B[d].count = n;
                if (n) {
                    DevGuard g(S[d].dev);
                    CK(ctx, cudaMemcpyAsync(B[d].base, B[0].ptr(es), n * es, cudaMemcpyDefault, S[d].stream));
                    ctx->stats.d2d_bytes += n * es;
                }
            }
            B[0].count = n;
            break;
        }
        case SKEL_XCHG_GATHER: {
            TRY(buf_grow(ctx, S[0], B[0], std::max<size_t>(n * es, 16), es, B[0].count * es, 0));
            TRY(join(ctx));
            for (int d = 1; d < D; ++d) {
                if (B[d].count) {
                    DevGuard g(S[0].dev);
                    CK(ctx, cudaMemcpyAsync(B[0].base + part_lo(v, d) * es, B[d].ptr(es), B[d].count * es,
                                            cudaMemcpyDefault, S[0].stream));
                    ctx->stats.d2d_bytes += B[d].count * es;
                }
                B[d].count = 0;
            }
            B[0].off = 0;
            B[0].count = n;
            break;
        }
        case SKEL_XCHG_ALLGATHER:
        case SKEL_XCHG_ALLREDUCE: {
            if (x == SKEL_XCHG_ALLREDUCE) {
                TRY(xchg_local(v, SKEL_XCHG_REDUCE_SCATTER, combine));
                TRY(join(ctx));
            }
            for (int d = 0; d < D; ++d) TRY(buf_grow(ctx, S[d], B[d], full_bytes(v), es, B[d].count * es, part_lo(v, d)));
            TRY(join(ctx));
            for (int d = 0; d < D; ++d) {
                DevGuard g(S[d].dev);
                for (int j = 0; j < D; ++j) {
                    if (j == d) continue;
                    const size_t cnt = want_count(v, SKEL_BLOCK, j);
                    if (!cnt) continue;
                    const size_t lo = part_lo(v, j);
                    CK(ctx, cudaMemcpyAsync(B[d].base + lo * es, B[j].base + lo * es, cnt * es, cudaMemcpyDefault,
                                            S[d].stream));
                    ctx->stats.d2d_bytes += cnt * es;
                }
                B[d].off = 0;
                B[d].count = n;
            }
            break;
        }
        case SKEL_XCHG_LOCAL_SLICE: {
            for (int d = 0; d < D; ++d) {
                B[d].off = part_lo(v, d);
                B[d].count = want_count(v, SKEL_BLOCK, d);
            }
            break;
        }
        case SKEL_XCHG_REDUCE_SCATTER: {
            for (int d = 0; d < D; ++d) {
                const size_t lo = part_lo(v, d), cnt = want_count(v, SKEL_BLOCK, d);
                B[d].off = lo;
                B[d].count = cnt;
                if (!cnt) continue;
                std::vector<const void *> src(D);
                std::vector<int> sdev(D);
                for (int j = 0; j < D; ++j) src[j] = B[j].base + lo * es, sdev[j] = S[j].dev;
                TRY(stage_remote(ctx, S[d], src, sdev, cnt * es));
                DevGuard g(S[d].dev);
                CK(ctx, launch_combine(B[d].base + lo * es, src.data(), D, cnt, v->dt, combine, S[d].stream));
                ctx->stats.kernel_launches++;
                ctx->stats.d2d_bytes += (D - 1) * cnt * es;
            }
            break;
        }
        case SKEL_XCHG_KEEP_ROOT: {
            for (int d = 1; d < D; ++d) B[d].count = 0;
            break;
        }
        case SKEL_XCHG_REDUCE: {
            std::vector<const void *> src(D);
            std::vector<int> sdev(D);
            for (int j = 0; j < D; ++j) src[j] = B[j].base, sdev[j] = S[j].dev;
            TRY(stage_remote(ctx, S[0], src, sdev, n * es));
            DevGuard g(S[0].dev);
            CK(ctx, launch_combine(B[0].base, src.data(), D, n, v->dt, combine, S[0].stream));
            ctx->stats.kernel_launches++;
            ctx->stats.d2d_bytes += (D - 1) * n * es;
            for (int d = 1; d < D; ++d) B[d].count = 0;
            B[0].off = 0;
            B[0].count = n;
            break;
        }
        default: break;
    }
    return join(ctx);
}

// Rank mode: this process holds logical device `rank`; NCCL moves the data,
// in place wherever NCCL allows it (part k at offset k*ceil(n/D) of a full
// buffer).
int xchg_rank(skel_vec_s *v, int x, skel_combine combine) {
    skel_ctx_s *ctx = v->ctx;
    const int D = ctx->D, r = ctx->rank;
    const size_t es = v->es, n = v->n, ps = part_size(n, D);
    Slot &s = ctx->slots[0];
    Buf &b = v->bufs[0];
    ncclComm_t c = ctx->comm;
    DevGuard g(s.dev);
    switch (x) {
        case SKEL_XCHG_SCATTER: {
            if (r == 0) TRY(buf_grow(ctx, s, b, full_bytes(v), es, n * es, 0));
            else if (b.cap < std::max<size_t>(ps * es, 16)) TRY(buf_grow(ctx, s, b, std::max<size_t>(ps * es, 16), es, 0, 0));
            b.off = 0;
            NK(ctx, ncclScatter(b.base, b.base, ps * es, ncclUint8, 0, c, s.stream));
            ctx->stats.nccl_bytes += ps * es * (r == 0 ? D : 1);
            b.count = want_count(v, SKEL_BLOCK, r);
            break;
        }
        case SKEL_XCHG_BROADCAST: {
            TRY(buf_grow(ctx, s, b, full_bytes(v), es, r == 0 ? n * es : 0, 0));
            NK(ctx, ncclBroadcast(b.base, b.base, n * es, ncclUint8, 0, c, s.stream));
            ctx->stats.nccl_bytes += n * es;
            b.off = 0;
            b.count = n;
            break;
        }
        case SKEL_XCHG_GATHER: {
            if (r == 0) TRY(buf_grow(ctx, s, b, full_bytes(v), es, b.count * es, 0));
            NK(ctx, ncclGather(b.ptr(es), b.base, ps * es, ncclUint8, 0, c, s.stream));
            ctx->stats.nccl_bytes += ps * es;
            b.count = r == 0 ? n : 0;
            b.off = 0;
            break;
        }
        case SKEL_XCHG_ALLGATHER: {
            TRY(buf_grow(ctx, s, b, full_bytes(v), es, b.count * es, part_lo(v, r) == std::min(n, r * ps) ? r * ps : 0));
            NK(ctx, ncclAllGather(b.base + r * ps * es, b.base, ps * es, ncclUint8, c, s.stream));
            ctx->stats.nccl_bytes += ps * es * D;
            b.off = 0;
            b.count = n;
            break;
        }
        case SKEL_XCHG_LOCAL_SLICE: {
            b.off = part_lo(v, r);
            b.count = want_count(v, SKEL_BLOCK, r);
            break;
        }
        case SKEL_XCHG_REDUCE_SCATTER: {
            NK(ctx, ncclReduceScatter(b.base, b.base + r * ps * es, ps, nccl_type(v->dt), nccl_op(combine), c,
                                      s.stream));
            ctx->stats.nccl_bytes += ps * es * D;
            b.off = r * ps;
            b.count = want_count(v, SKEL_BLOCK, r);
            break;
        }
        case SKEL_XCHG_KEEP_ROOT: {
            if (r != 0) b.count = 0;
            break;
        }
        case SKEL_XCHG_REDUCE: {
            NK(ctx, ncclReduce(b.base, b.base, n, nccl_type(v->dt), nccl_op(combine), 0, c, s.stream));
            ctx->stats.nccl_bytes += n * es;
            b.count = r == 0 ? n : 0;
            break;
        }
        case SKEL_XCHG_ALLREDUCE: {
            NK(ctx, ncclAllReduce(b.base, b.base, n, nccl_type(v->dt), nccl_op(combine), c, s.stream));
            ctx->stats.nccl_bytes += n * es;
            break;
        }
        default: break;
    }
    return SKEL_OK;
}

int set_distribution(skel_vec_s *v, skel_dist dist, skel_combine combine) {
    skel_ctx_s *ctx = v->ctx;
    TRY(wait_dl(v));  // exchanges rewrite the buffers
    const int x = plan_exchange(v->dist, dist, combine);
    if (x < 0) return fail(ctx, SKEL_ERR_STATE, "a combine merges per-device copies: the vector must be SKEL_COPY");
    if (combine != SKEL_COMBINE_NONE && v->dt == SKEL_DT_OPAQUE)
        return fail(ctx, SKEL_ERR_TYPE, "combine needs a numeric dtype (skel_vector_set_dtype)");
    if (!v->dev_valid && combine == SKEL_COMBINE_NONE && !partial_mirror(v)) {  // host-only data: free relayout
        v->dist = dist;
        return SKEL_OK;
    }
    TRY(ensure_device(v));
    if (x == SKEL_XCHG_NONE) {
        v->dist = dist;
        return SKEL_OK;
    }
    const bool diverged = v->diverged;
    if (ctx->D == 1) {
        // one device: every distribution is the same storage
        Buf &b = v->bufs[0];
        b.off = 0;
        b.count = v->n;
    } else if (ctx->rank_mode) {
        TRY(xchg_rank(v, x, combine));
    } else {
        TRY(xchg_local(v, x, combine));
    }
    v->dist = dist;
    v->dev_valid = true;
    if (combine != SKEL_COMBINE_NONE || diverged) device_wrote(v);
    v->diverged = false;
    return SKEL_OK;
}

// ---- user-defined combine ---------------------------------
// The paper's combine is "element-wise add"; here any associative
// user function T f(T, T) given as source text (an NVRTC-built Zip module) merges
// the copies element-wise, folded in device order 0..D-1 (non-commutative f ok).

int ew_grid(const Slot &s, size_t chunks, int block, int per_thread = 1);
int ensure_ws(skel_ctx_s *ctx, Slot &s, size_t bytes);

// Kernel launches of the skeleton templates: as a programmatic dependent of
// the previous kernel on the stream (cudaLaunchAttributeProgrammaticStreamSerialization).
// Every such kernel starts with griddepcontrol.wait (prelude.cuh skel::pdl_wait:
// it touches no memory before the previous kernel has completed and its writes
// are visible) and then lets its own dependents be scheduled, so the next
// kernel's CTAs are placed during this one's last wave and the launch gap
// between consecutive skeletons disappears.  A non-kernel predecessor (copy,
// event wait) or a kernel that never triggers keeps the ordinary ordering.
// SKEL_PDL=0: plain launches.
bool pdl_enabled() {
    static const bool pdl = [] {
        const char *e = getenv("SKEL_PDL");
        return !(e && atoi(e) == 0);
    }();
    return pdl;
}
cudaError_t launch_dependent(const void *fn, dim3 grid, dim3 block, void **params, cudaStream_t st,
                             size_t smem = 0) {
    if (!pdl_enabled()) return cudaLaunchKernel(fn, grid, block, params, smem, st);
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = grid;
    cfg.blockDim = block;
    cfg.dynamicSmemBytes = smem;
    cfg.stream = st;
    cudaLaunchAttribute at[1];
    at[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    at[0].val.programmaticStreamSerializationAllowed = 1;
    cfg.attrs = at;
    cfg.numAttrs = 1;
    return cudaLaunchKernelExC(&cfg, fn, params);
}

// one Zip launch out[i] = f(a[i], b[i]) on raw device pointers (out may alias a or b)
int zip_raw(skel_ctx_s *ctx, Module *m, Slot &s, const void *pa, const void *pb, void *po, uint64_t cnt) {
    if (!cnt) return SKEL_OK;
    std::vector<unsigned char> abuf(std::max<uint64_t>(m->sig[7], 16), 0);
    const int block = (int)m->sig[9];
    const uint64_t E = m->sig[8];
    int vec_ok = al16(pa) && al16(pb) && al16(po);
    const size_t chunks = vec_ok ? std::max<uint64_t>(cnt / E, 1) : cnt;
    const int grid = ew_grid(s, chunks, block, vec_ok && E > 1 ? std::max<int>(1, (int)m->sig[10]) : 1);
    void *params[] = {&pa, &pb, &po, &cnt, &vec_ok, abuf.data()};
    DevGuard g(s.dev);
    CK(ctx, launch_dependent((const void *)m->k_main, dim3(grid), dim3(block), params, s.stream));
    ctx->stats.kernel_launches++;
    return SKEL_OK;
}

// dst = f(...f(f(src[0], src[1]), src[2])..., src[D-1]) over cnt elements on slot s
int fold_raw(skel_ctx_s *ctx, Module *m, Slot &s, const std::vector<const char *> &src, char *dst, uint64_t cnt) {
    TRY(zip_raw(ctx, m, s, src[0], src[1], dst, cnt));
    for (size_t j = 2; j < src.size(); ++j) TRY(zip_raw(ctx, m, s, dst, src[j], dst, cnt));
    return SKEL_OK;
}

int set_distribution_fn(skel_vec_s *v, skel_dist dist, const char *src) {
    skel_ctx_s *ctx = v->ctx;
    TRY(wait_dl(v));
    if (v->dist != SKEL_COPY) return fail(ctx, SKEL_ERR_STATE, "a combine merges per-device copies: the vector must be SKEL_COPY");
    Module *m = nullptr;
    TRY(get_module(ctx, Kind::Zip, src, &m));
    if (m->sig[6] != 0) return fail(ctx, SKEL_ERR_TYPE, "a combine function takes exactly two parameters");
    if (m->sig[3] != v->es || m->sig[4] != v->es || m->sig[5] != v->es)
        return fail(ctx, SKEL_ERR_TYPE, "combine function must have the form T f(T, T) with sizeof(T) = element size");
    TRY(ensure_device(v));
    const int D = ctx->D;
    const size_t es = v->es, n = v->n;
    if (D == 1) {  // one copy: nothing to merge
        Buf &b = v->bufs[0];
        b.off = 0;
        b.count = n;
    } else if (!ctx->rank_mode) {
        auto &S = ctx->slots;
        auto &B = v->bufs;
        TRY(join(ctx));
        // operands of device d's fold, staged locally when P2P is missing
        auto operands = [&](int d, size_t lo, size_t cnt, std::vector<const char *> &srcs) -> int {
            std::vector<const void *> src(D);
            std::vector<int> sdev(D);
            for (int j = 0; j < D; ++j) src[j] = B[j].base + lo * es, sdev[j] = S[j].dev;
            TRY(stage_remote(ctx, S[d], src, sdev, cnt * es));
            srcs.resize(D);
            for (int j = 0; j < D; ++j) srcs[j] = static_cast<const char *>(src[j]);
            return SKEL_OK;
        };
        if (dist == SKEL_SINGLE) {
            std::vector<const char *> srcs;
            TRY(operands(0, 0, n, srcs));
            TRY(fold_raw(ctx, m, S[0], srcs, B[0].base, n));
            ctx->stats.d2d_bytes += (D - 1) * n * es;
            TRY(join(ctx));
            for (int d = 1; d < D; ++d) B[d].count = 0;
            B[0].off = 0;
            B[0].count = n;
        } else {
            // device d merges part d of every copy into part d of its own copy; for
            // d >= 2 its own copy is a later operand of the fold, so the fold runs in
            // the slot's workspace and is copied over afterwards
            for (int d = 0; d < D; ++d) {
                const size_t lo = part_lo(v, d), cnt = want_count(v, SKEL_BLOCK, d);
                if (!cnt) continue;
                std::vector<const char *> srcs;
                TRY(operands(d, lo, cnt, srcs));
                char *own = B[d].base + lo * es;
                if (d < 2) {
                    TRY(fold_raw(ctx, m, S[d], srcs, own, cnt));
                } else {
                    TRY(ensure_ws(ctx, S[d], cnt * es + 256));
                    TRY(fold_raw(ctx, m, S[d], srcs, S[d].ws, cnt));
                    DevGuard g(S[d].dev);
                    CK(ctx, cudaMemcpyAsync(own, S[d].ws, cnt * es, cudaMemcpyDeviceToDevice, S[d].stream));
                }
                ctx->stats.d2d_bytes += (D - 1) * cnt * es;
            }
            TRY(join(ctx));
            for (int d = 0; d < D; ++d) {
                B[d].off = part_lo(v, d);
                B[d].count = want_count(v, SKEL_BLOCK, d);
            }
            if (dist == SKEL_COPY) TRY(xchg_local(v, SKEL_XCHG_ALLGATHER, SKEL_COMBINE_NONE));
        }
    } else {
        // one process per GPU: every rank's part r of its copy is gathered on rank r
        // (D gathers, one per root), then folded there in rank order
        Slot &s = ctx->slots[0];
        Buf &b = v->bufs[0];
        const int r = ctx->rank;
        const size_t ps = part_size(n, D);
        const size_t piece = dist == SKEL_SINGLE ? n : ps;
        TRY(ensure_ws(ctx, s, (size_t)D * piece * es + 256));
        char *stage = s.ws;
        DevGuard g(s.dev);
        if (dist == SKEL_SINGLE) {
            NK(ctx, ncclGather(b.base, stage, n * es, ncclUint8, 0, ctx->comm, s.stream));
            ctx->stats.nccl_bytes += n * es;
        } else {
            for (int j = 0; j < D; ++j) {
                NK(ctx, ncclGather(b.base + (size_t)j * ps * es, stage, ps * es, ncclUint8, j, ctx->comm, s.stream));
                ctx->stats.nccl_bytes += ps * es;
            }
        }
        const size_t lo = dist == SKEL_SINGLE ? 0 : part_lo(v, r);
        const size_t cnt = dist == SKEL_SINGLE ? (r == 0 ? n : 0) : want_count(v, SKEL_BLOCK, r);
        if (cnt) {
            std::vector<const char *> srcs(D);
            for (int j = 0; j < D; ++j) srcs[j] = stage + (size_t)j * piece * es;
            TRY(fold_raw(ctx, m, s, srcs, b.base + lo * es, cnt));
        }
        b.off = lo;
        b.count = cnt;
        if (dist == SKEL_COPY) TRY(xchg_rank(v, SKEL_XCHG_ALLGATHER, SKEL_COMBINE_NONE));
    }
    v->dist = dist;
    v->dev_valid = true;
    device_wrote(v);
    v->diverged = false;
    return SKEL_OK;
}

// ---- Arguments (§III-C) ------------------------------------------------------
int check_args(skel_ctx_s *ctx, const Module *m, const skel_arg *args, int nargs) {
    const int want = (int)m->sig[6];
    if (nargs != want)
        return fail(ctx, SKEL_ERR_TYPE, "user function takes " + std::to_string(want) + " extra argument(s), " +
                                            std::to_string(nargs) + " given");
    for (int i = 0; i < nargs; ++i) {
        const uint64_t size = m->sig[16 + 4 * i], isptr = m->sig[18 + 4 * i];
        if (args[i].kind == SKEL_ARG_VECTOR) {
            if (!isptr) return fail(ctx, SKEL_ERR_TYPE, "argument " + std::to_string(i) + ": vector for a by-value parameter");
            if (!args[i].vec || args[i].vec->ctx != ctx) return fail(ctx, SKEL_ERR_ARG, "argument " + std::to_string(i) + ": bad vector");
        } else if (args[i].kind == SKEL_ARG_SCALAR) {
            if (args[i].size != size || !args[i].data)
                return fail(ctx, SKEL_ERR_TYPE, "argument " + std::to_string(i) + ": " + std::to_string(args[i].size) +
                                                    " bytes given, parameter has " + std::to_string(size));
        } else {
            return fail(ctx, SKEL_ERR_ARG, "argument " + std::to_string(i) + ": bad kind");
        }
    }
    for (int i = 0; i < nargs; ++i)
        if (args[i].kind == SKEL_ARG_VECTOR) {
            TRY(ensure_device(args[i].vec));
            TRY(wait_dl(args[i].vec));  // a side-effect Map may write it
        }
    return SKEL_OK;
}
void pack_args(const Module *m, const skel_arg *args, int nargs, size_t li, std::vector<unsigned char> &buf) {
    buf.assign(m->sig[7], 0);
    for (int i = 0; i < nargs; ++i) {
        const uint64_t off = m->sig[19 + 4 * i];
        if (args[i].kind == SKEL_ARG_VECTOR) {
            skel_vec_s *av = args[i].vec;
            void *p = av->bufs[li].ptr(av->es);
            memcpy(&buf[off], &p, sizeof p);
        } else {
            memcpy(&buf[off], args[i].data, args[i].size);
        }
    }
}

int prepare_output(skel_vec_s *out, size_t n, skel_dist dist, bool same_as_input) {
    TRY(wait_dl(out));
    if (!same_as_input) {
        if (out->n != n) {  // resize: the output gets the input's length
            out->n = n;
            if (out->host) {
                cudaFreeHost(out->host);
                out->host = nullptr;
            }
        }
        out->dist = dist;
        TRY(place(out, dist));
    }
    out->dev_valid = true;
    device_wrote(out);
    out->diverged = false;
    return SKEL_OK;
}

// grid of the element-wise kernels: one chunk per thread, or -- when the kernel
// keeps `per_thread` chunks in flight per thread (vectorised path) -- just
// enough threads to give each of them that many, but never less than one full
// resident wave while there is work for it; capped at `waves` resident waves
// (a grid-stride loop covers the rest)
int ew_grid(const Slot &s, size_t chunks, int block, int per_thread) {
    static const int waves = [] {
        const char *e = getenv("SKEL_EW_WAVES");  // tuning hook: grid = SMs x (2048/block) x waves
        return e ? std::max(1, atoi(e)) : 32;
    }();
    static const int pt_env = [] {
        const char *e = getenv("SKEL_EW_PER_THREAD");  // tuning hook: chunks per thread for the sizing
        return e ? atoi(e) : 0;
    }();
    if (pt_env > 0 && per_thread > 1) per_thread = std::min(per_thread, pt_env);
    size_t g = (chunks + block - 1) / block;
    if (per_thread > 1) {
        const size_t resident = (size_t)s.sms * (2048 / block);
        const size_t gu = (chunks + (size_t)block * per_thread - 1) / ((size_t)block * per_thread);
        g = std::max(gu, std::min(g, resident));
    }
    const size_t cap = (size_t)s.sms * (2048 / block) * waves;
    g = std::min(g, cap);
    return (int)std::max<size_t>(g, 1);
}

// Element-wise grid policy of a module (Module::ew_policy): 0 = UNROLL chunks
// in flight per thread (bandwidth-bound functions), 1 = one chunk per thread,
// 2 = one element per thread through the scalar path (compute-bound, divergent
// functions: finer work items even out the lanes of a warp), 3 = one chunk per
// thread with the low-register kernel (small vectors: twice the CTAs per SM,
// so a single-wave launch), 4 = the scalar path through the low-register kernel,
// 5 = the same over half a grid: every thread takes elements i and i + n/2
// (for a divergent function two items of uncorrelated cost per lane even out a
// warp's lanes better than one: Mandelbrot rows y and y + H/2, 7% faster).  Decided once per
// module, size class (log2 of the chunk count) and set of scalar arguments (up
// to four per class), at the first launch of that class and set, by timing the policies in `mask` on a SAMPLE of that launch's data
// copied to scratch memory -- never on the user's buffers,
// so no user launch runs with a losing policy and nothing the user owns is
// written twice.  The sample: 256 evenly spread blocks of the input(s), up to
// 256 MB of operands in all (the whole vector if smaller), each policy timed
// three times (best of three); an index Map samples four contiguous index
// ranges spread over [0, n).  Functions with pointer
// (vector) arguments may have side effects and are not sampled: they take the
// mask's lowest policy.  The lowest policy is also the default another must
// beat by 3%.
bool has_ptr_args(const Module *m) {
    for (uint64_t i = 0; i < m->sig[6] && i < 32; ++i)
        if (m->sig[18 + 4 * i]) return true;
    return false;
}

int ew_decide(skel_ctx_s *ctx, Module *m, Slot &s, Kind kind, const void *pa, size_t esa, const void *pb, size_t esb,
              size_t eso, uint64_t cnt, uint64_t base, std::vector<unsigned char> &abuf, unsigned mask, int *policy) {
    int pol[Module::kPolicies], P = 0;
    for (int p = 0; p < Module::kPolicies; ++p)
        if (mask & (1u << p)) pol[P++] = p;
    *policy = pol[0];
    const uint64_t E0 = std::max<uint64_t>(m->sig[8], 1);
    const int cls = 64 - __builtin_clzll((unsigned long long)std::max<uint64_t>(cnt / E0, 1));
    // the scalar arguments can change a function's cost profile (Mandelbrot's
    // iteration cap: at 4096 the periodicity check makes the work far more
    // uneven than at 256), so they are part of the key -- up to kArgKeys
    // argument sets per size class; later sets reuse a decided one (no trials
    // for a function whose argument changes at every launch)
    constexpr int kArgKeys = 4;
    uint64_t ah = 1469598103934665603ull;  // FNV-1a of the packed scalar arguments
    for (unsigned char c : abuf) ah = (ah ^ c) * 1099511628211ull;
    const auto key = std::make_pair(cls, ah);
    char tag[32];
    snprintf(tag, sizeof tag, "cc%d_sm%d", s.cc, s.sms);
    if (!m->policy_loaded) {
        m->policy_loaded = true;
        if (!m->policy_path.empty()) {
            std::ifstream f(m->policy_path);
            std::string t;
            int c, p;
            unsigned long long h;
            while (f >> t >> c >> h >> p)
                if (t == tag && p >= 0 && p < Module::kPolicies && (mask >> p & 1u))
                    m->ew_policy.emplace(std::make_pair(c, (uint64_t)h), p);
        }
    }
    auto known = m->ew_policy.find(key);
    if (known != m->ew_policy.end()) {
        *policy = known->second;
        return SKEL_OK;
    }
    {
        auto it = m->ew_policy.lower_bound(std::make_pair(cls, (uint64_t)0));
        int seen = 0;
        int first = -1;
        for (; it != m->ew_policy.end() && it->first.first == cls; ++it, ++seen)
            if (first < 0) first = it->second;
        if (seen >= kArgKeys) {
            *policy = first;
            return SKEL_OK;
        }
    }
    cudaStreamCaptureStatus cs = cudaStreamCaptureStatusNone;
    cudaStreamIsCapturing(s.stream, &cs);
    if (cs != cudaStreamCaptureStatusNone || eso == 0 || has_ptr_args(m) || P < 2) {
        if (cs == cudaStreamCaptureStatusNone) m->ew_policy[key] = pol[0];
        return SKEL_OK;
    }
    const uint64_t E = m->sig[8];
    const int block = (int)m->sig[9];
    const int unroll = std::max<int>(1, (int)m->sig[10]);
    // sample: up to 256 MB of operands -- more than the 126 MB L2, so the trials
    // see the memory system the full launch sees (an L2-resident sample once
    // made the scalar path look as fast as the vector path for a Zip)
    constexpr uint64_t kSampleBytes = 256ull << 20, kBlocks = 256;
    const uint64_t kSample = std::max<uint64_t>(kSampleBytes / std::max<size_t>(esa + esb + eso, 1), 4096);
    if (cnt > kSample && (mask & 56u)) {
        // the low-register kernel is a small-vector policy: judged only where the
        // sample IS the launch (at 2^30 a sample once preferred it by noise, 1.7%
        // slower at full size)
        mask &= ~56u;
        P = 0;
        for (int p = 0; p < Module::kPolicies; ++p)
            if (mask & (1u << p)) pol[P++] = p;
    }
    uint64_t ns = std::min<uint64_t>(cnt, kSample) / E * E;
    if (ns == 0) return SKEL_OK;  // decide at a larger launch
    const size_t oa = 0, ob = align_up(ns * esa, 256), oo = ob + align_up(pb ? ns * esb : 0, 256);
    const size_t per_copy = oo + align_up(ns * eso, 256);
    // a sample smaller than L2 is replicated so that consecutive trial launches
    // touch different copies and stream from HBM, as a user's launches on
    // distinct vectors would (an L2-resident sample hides the memory behaviour)
    const int copies = per_copy < (128ull << 20) ? (int)std::min<uint64_t>(16, (256ull << 20) / per_copy) : 1;
    TRY(scratch(ctx, s, per_copy * copies));
    char *sa = s.scratch + oa, *sb = s.scratch + ob, *so = s.scratch + oo;
    DevGuard g(s.dev);
    std::vector<std::pair<uint64_t, uint64_t>> ranges;  // index Map: (base, count) per launch
    if (kind == Kind::Idx && cnt <= kSample) {
        ranges.push_back({base, cnt});  // the trial launch is the user's launch
    } else if (kind == Kind::Idx) {
        // four pieces spread over the index range (a divergent function's cost
        // varies along it, e.g. the rows of a Mandelbrot image)
        const uint64_t part = ns / 4 / E * E;
        for (int r = 0; r < 4 && part; ++r) {
            const uint64_t lo = std::min<uint64_t>(cnt - part, (cnt / 4) * r + cnt / 8 - std::min(cnt / 8, part / 2));
            ranges.push_back({base + lo, part});
        }
        if (ranges.empty()) ranges.push_back({base, ns});
    } else if (cnt <= kSample) {
        CK(ctx, cudaMemcpyAsync(sa, pa, ns * esa, cudaMemcpyDeviceToDevice, s.stream));
        if (pb) CK(ctx, cudaMemcpyAsync(sb, pb, ns * esb, cudaMemcpyDeviceToDevice, s.stream));
        ranges.push_back({0, ns});
    } else {
        const uint64_t blk = std::max<uint64_t>(E, ns / kBlocks / E * E), nblk = ns / blk;
        const uint64_t stride = cnt / nblk;  // >= blk
        CK(ctx, cudaMemcpy2DAsync(sa, blk * esa, pa, stride * esa, blk * esa, nblk, cudaMemcpyDeviceToDevice,
                                  s.stream));
        if (pb)
            CK(ctx, cudaMemcpy2DAsync(sb, blk * esb, pb, stride * esb, blk * esb, nblk, cudaMemcpyDeviceToDevice,
                                      s.stream));
        ns = blk * nblk;
        ranges.push_back({0, ns});
    }
    for (int k = 1; k < copies && kind != Kind::Idx; ++k) {  // the replicas of the inputs
        CK(ctx, cudaMemcpyAsync(sa + k * per_copy, sa, ns * esa, cudaMemcpyDeviceToDevice, s.stream));
        if (pb) CK(ctx, cudaMemcpyAsync(sb + k * per_copy, sb, ns * esb, cudaMemcpyDeviceToDevice, s.stream));
    }
    int rot = 0;  // the copy the next trial launch uses
    constexpr int kRounds = 3;
    cudaEvent_t ev[2 * Module::kPolicies * kRounds] = {};
    for (auto &e : ev) CK(ctx, cudaEventCreate(&e));
    auto launch = [&](int policy) -> int {
        const size_t off = (size_t)(rot++ % copies) * per_copy;
        for (auto &rg : ranges) {
            uint64_t n = rg.second, b0 = rg.first;
            const size_t chunks = std::max<uint64_t>(n / E, 1);
            const bool scalar = policy == 2 || policy == 4 || policy == 5;
            int vk = scalar ? 0 : 1;
            const void *qa = sa + off, *qb = pb ? (const void *)(sb + off) : nullptr;
            void *qo = so + off;
            int grid;
            if (kind == Kind::Idx) {
                grid = ew_grid(s, scalar ? n : chunks, block, policy == 5 ? 2 : 1);
                void *params[] = {&qo, &n, &b0, &vk, abuf.data()};
                CK(ctx, cudaLaunchKernel((const void *)m->k_main, dim3(grid), dim3(block), params, 0, s.stream));
            } else {
                grid = scalar ? ew_grid(s, n, block, policy == 5 ? 2 : 1)
                              : ew_grid(s, chunks, block, policy == 0 ? unroll : 1);
                void *params[] = {&qa, &qb, &qo, &n, &vk, abuf.data()};
                const void *kf = policy >= 3 ? (const void *)m->k_main_u1 : (const void *)m->k_main;
                CK(ctx, cudaLaunchKernel(kf, dim3(grid), dim3(block), params, 0, s.stream));
            }
        }
        return SKEL_OK;
    };
    // warm every policy once (first touch of the module on this device) and time
    // that pass, so that short launches are measured in repetitions of about
    // 200 us (a lone 25 us launch is at the mercy of launch gaps)
    CK(ctx, cudaEventRecord(ev[0], s.stream));
    for (int p = 0; p < P; ++p) TRY(launch(pol[p]));
    CK(ctx, cudaEventRecord(ev[1], s.stream));
    CK(ctx, cudaEventSynchronize(ev[1]));
    float warm = 0;
    CK(ctx, cudaEventElapsedTime(&warm, ev[0], ev[1]));
    const int reps = std::max(1, std::min(16, (int)(0.2f / std::max(warm / P, 1e-3f))));
    for (int k = 0; k < kRounds * P; ++k) {
        CK(ctx, cudaEventRecord(ev[2 * k], s.stream));
        for (int r = 0; r < reps; ++r) TRY(launch(pol[k % P]));
        CK(ctx, cudaEventRecord(ev[2 * k + 1], s.stream));
    }
    CK(ctx, cudaEventSynchronize(ev[2 * kRounds * P - 1]));
    float best_t[Module::kPolicies];
    for (int p = 0; p < P; ++p) best_t[p] = 3.0e38f;
    for (int k = 0; k < kRounds * P; ++k) {
        float t = 0;
        CK(ctx, cudaEventElapsedTime(&t, ev[2 * k], ev[2 * k + 1]));
        best_t[k % P] = std::min(best_t[k % P], t);
    }
    for (auto &e : ev) cudaEventDestroy(e);
    int b = 0;
    for (int p = 1; p < P; ++p)
        if (best_t[p] < 0.97f * best_t[0] && best_t[p] < best_t[b]) b = p;
    m->ew_policy[key] = pol[b];
    if (!m->policy_path.empty()) {  // one short O_APPEND write: concurrent ranks do not interleave
        char line[96];
        const int len = snprintf(line, sizeof line, "%s %d %llu %d\n", tag, cls, (unsigned long long)ah, pol[b]);
        const int fd = open(m->policy_path.c_str(), O_WRONLY | O_CREAT | O_APPEND, 0644);
        if (fd >= 0) {
            if (write(fd, line, (size_t)len) != len) { /* a lost line only costs a later trial */ }
            close(fd);
        }
    }
    if (getenv("SKEL_LOG")) {
        fprintf(stderr, "[skel] grid policy, size class %d, %d x %d reps:", cls, (int)ranges.size(), reps);
        for (int p = 0; p < P; ++p) fprintf(stderr, " p%d %.4f ms", pol[p], best_t[p] / reps);
        fprintf(stderr, " -> p%d\n", pol[b]);
    }
    ctx->stats.kernel_launches += (uint64_t)(kRounds * P * reps + P) * ranges.size();
    *policy = pol[b];
    return SKEL_OK;
}

int run_ew(skel_ctx_s *ctx, Kind kind, const char *src, skel_vec_s *a, skel_vec_s *b, skel_vec_s *out,
           const skel_arg *args, int nargs) {
    Module *m = nullptr;
    TRY(get_module(ctx, kind, src, &m));
    const uint64_t rsz = m->sig[3];
    if (m->sig[4] != a->es)
        return fail(ctx, SKEL_ERR_TYPE, "element size " + std::to_string(a->es) + " != sizeof(parameter 0) = " +
                                            std::to_string(m->sig[4]));
    if (b && m->sig[5] != b->es)
        return fail(ctx, SKEL_ERR_TYPE, "element size of the second vector != sizeof(parameter 1)");
    if (rsz == 0 && kind == Kind::Zip) return fail(ctx, SKEL_ERR_TYPE, "zip needs a non-void function");
    if (rsz != 0 && !out) return fail(ctx, SKEL_ERR_ARG, "non-void function needs an output vector");
    if (rsz != 0 && out->es != rsz)
        return fail(ctx, SKEL_ERR_TYPE, "output element size " + std::to_string(out->es) + " != sizeof(result) = " +
                                            std::to_string(rsz));
    TRY(check_args(ctx, m, args, nargs));
    TRY(ensure_device(a));
    if (b) {
        if (b->dist != a->dist) TRY(set_distribution(b, a->dist, SKEL_COMBINE_NONE));
        TRY(ensure_device(b));
    }
    if (rsz != 0) TRY(prepare_output(out, a->n, a->dist, out == a || out == b));
    const int block = (int)m->sig[9];
    const uint64_t E = m->sig[8];
    std::vector<unsigned char> abuf;
    for (size_t li = 0; li < ctx->slots.size(); ++li) {
        Slot &s = ctx->slots[li];
        uint64_t cnt = a->bufs[li].count;
        if (!cnt) continue;
        const void *pa = a->bufs[li].ptr(a->es);
        const void *pb = b ? b->bufs[li].ptr(b->es) : nullptr;
        void *po = (rsz != 0) ? out->bufs[li].ptr(out->es) : nullptr;
        int vec_ok = al16(pa) && (!pb || al16(pb)) && (!po || al16(po));
        pack_args(m, args, nargs, li, abuf);
        const size_t chunks = vec_ok ? std::max<uint64_t>(cnt / E, 1) : cnt;
        const int unroll = std::max<int>(1, (int)m->sig[10]);
        DevGuard g(s.dev);
        // grid policy (Module::ew_policy): decided on a sample at the module's first launch
        int policy = 0;
        if (vec_ok && E > 1 && unroll > 1)
            TRY(ew_decide(ctx, m, s, kind, pa, a->es, pb, b ? b->es : 0, rsz, cnt, 0, abuf,
                          m->k_main_u1 ? 0x3Fu : 0x7u, &policy));
        // policy 2: the scalar path, one element per thread; 3: one chunk per thread
        // through the low-register kernel; 4: the scalar path through it; 5: the
        // same with two elements per thread (grid-stride over half a grid)
        const bool scalar = policy == 2 || policy == 4 || policy == 5;
        int vk = scalar ? 0 : vec_ok;
        const int grid = scalar ? ew_grid(s, cnt, block, policy == 5 ? 2 : 1)
                                : ew_grid(s, chunks, block, policy == 0 && vec_ok && E > 1 ? unroll : 1);
        void *params[] = {&pa, &pb, &po, &cnt, &vk, abuf.data()};
        const void *kf = policy >= 3 ? (const void *)m->k_main_u1 : (const void *)m->k_main;
        CK(ctx, launch_dependent(kf, dim3(grid), dim3(block), params, s.stream));
        ctx->stats.kernel_launches++;
    }
    if (rsz != 0) {
        out->dev_valid = true;
        device_wrote(out);
    }
    return SKEL_OK;
}

// ---- fused copy->block combine + Zip + block->copy (NEXT-1) ---------------------
int ensure_ws(skel_ctx_s *ctx, Slot &s, size_t bytes);
// rank mode: a stream-ordered barrier over all ranks (a one-word all-reduce)
int rank_barrier(skel_ctx_s *ctx, Slot &s) {
    DevGuard g(s.dev);
    NK(ctx, ncclAllReduce(s.counters + 8, s.counters + 8, 1, ncclInt32, ncclSum, ctx->comm, s.stream));
    return SKEL_OK;
}

void close_peers(Buf &b) {
    for (size_t r = 0; r < b.peers.size(); ++r)
        if (b.peers[r] && b.peers[r] != b.base) cudaIpcCloseMemHandle(b.peers[r]);
    b.peers.clear();
    b.peers_of = nullptr;
}

// rank mode: open every rank's allocation of this buffer through CUDA IPC
// (collective: all ranks call it for the same vector)
int ipc_peers(skel_ctx_s *ctx, Slot &s, Buf &b) {
    if (b.peers_of == b.base && (int)b.peers.size() == ctx->D) return SKEL_OK;
    close_peers(b);
    DevGuard g(s.dev);
    TRY(sync_all(ctx));
    cudaIpcMemHandle_t mine;
    CK(ctx, cudaIpcGetMemHandle(&mine, b.base));
    const size_t hb = sizeof(cudaIpcMemHandle_t);
    TRY(ensure_ws(ctx, s, std::max<size_t>(s.ws_cap, hb * (ctx->D + 1))));
    // stream-ordered: the all-gather below runs on s.stream
    CK(ctx, cudaMemcpyAsync(s.ws, &mine, hb, cudaMemcpyHostToDevice, s.stream));
    NK(ctx, ncclAllGather(s.ws, s.ws + hb, hb, ncclUint8, ctx->comm, s.stream));
    std::vector<cudaIpcMemHandle_t> all(ctx->D);
    CK(ctx, cudaMemcpyAsync(all.data(), s.ws + hb, hb * ctx->D, cudaMemcpyDeviceToHost, s.stream));
    CK(ctx, cudaStreamSynchronize(s.stream));
    b.peers.assign(ctx->D, nullptr);
    for (int r = 0; r < ctx->D; ++r) {
        if (r == ctx->rank) {
            b.peers[r] = b.base;
            continue;
        }
        void *p = nullptr;
        CK(ctx, cudaIpcOpenMemHandle(&p, all[r], cudaIpcMemLazyEnablePeerAccess));
        b.peers[r] = static_cast<char *>(p);
    }
    b.peers_of = b.base;
    return SKEL_OK;
}

// rank mode: do all ranks report ok?  (a one-word MIN all-reduce, then a sync)
int rank_agree(skel_ctx_s *ctx, Slot &s, int ok, int *all_ok) {
    DevGuard g(s.dev);
    int v = ok ? 1 : 0;
    CK(ctx, cudaMemcpyAsync(s.counters + 9, &v, sizeof v, cudaMemcpyHostToDevice, s.stream));
    NK(ctx, ncclAllReduce(s.counters + 9, s.counters + 9, 1, ncclInt32, ncclMin, ctx->comm, s.stream));
    CK(ctx, cudaMemcpyAsync(&v, s.counters + 9, sizeof v, cudaMemcpyDeviceToHost, s.stream));
    CK(ctx, cudaStreamSynchronize(s.stream));
    *all_ok = v;
    return SKEL_OK;
}

// rank mode, SKEL_NCCL_WINDOWS=1: move vector v's buffer into an
// NCCL symmetric window -- ncclMemAlloc (VMM memory NCCL can map on every
// rank), the data copied over, ncclCommWindowRegister(NCCL_WIN_COLL_SYMMETRIC)
// -- and read from the window every rank's load/store address (the LSA flat
// mapping) and, with a device communicator that has multimem, the buffer's
// multicast address.  Collective: every rank calls it for the same vector.
// *ok = false (and SKEL_OK) on any failure, agreed by all ranks before the
// collective registration; the caller then opens the peers with CUDA IPC.
int win_setup(skel_ctx_s *ctx, Slot &s, skel_vec_s *v, bool *ok) {
    *ok = false;
    Buf &b = v->bufs[0];
    if (ctx->wins.count(b.base)) {
        *ok = true;
        return SKEL_OK;
    }
    const size_t es = v->es;
    const size_t size = align_up(std::max<size_t>(full_bytes(v), 1), NCCL_WIN_REQUIRED_ALIGNMENT);
    DevGuard g(s.dev);
    TRY(sync_all(ctx));
    void *p = nullptr;
    const bool alloc_ok = ncclMemAlloc(&p, size) == ncclSuccess && p;
    int all = 0;
    TRY(rank_agree(ctx, s, alloc_ok, &all));
    if (!all) {
        if (alloc_ok) ncclMemFree(p);
        if (getenv("SKEL_LOG")) fprintf(stderr, "[skel] NCCL symmetric window: ncclMemAlloc refused on some rank\n");
        return SKEL_OK;
    }
    char *nb = static_cast<char *>(p);
    if (b.count) CK(ctx, cudaMemcpyAsync(nb + b.off * es, b.base + b.off * es, b.count * es, cudaMemcpyDeviceToDevice,
                                         s.stream));
    CK(ctx, cudaStreamSynchronize(s.stream));
    close_peers(b);
    TRY(dev_free(ctx, s, b.base));
    b.base = nb;
    b.cap = size;
    ctx->nccl_mem.insert(nb);
    ncclWindow_t win = nullptr;
    const bool reg_ok = ncclCommWindowRegister(ctx->comm, nb, size, &win, NCCL_WIN_COLL_SYMMETRIC) == ncclSuccess;
    TRY(rank_agree(ctx, s, reg_ok, &all));
    if (!all) {
        if (reg_ok) ncclCommWindowDeregister(ctx->comm, win);
        if (getenv("SKEL_LOG"))
            fprintf(stderr, "[skel] NCCL symmetric window: ncclCommWindowRegister refused on some rank\n");
        return SKEL_OK;  // the buffer stays an ncclMemAlloc one; peers through IPC will fail -> unfused
    }
    ncclWindow_vidmem wv;
    CK(ctx, cudaMemcpy(&wv, win, sizeof wv, cudaMemcpyDefault));
    WinRec rec;
    rec.win = win;
    rec.size = size;
    const size_t four_g = (size_t)1 << 32;
    for (int r = 0; r < ctx->D; ++r) rec.peers.push_back(wv.lsaFlatBase + (size_t)r * wv.stride4G * four_g);
    if (ctx->devcomm_state < 0) {  // one device communicator per context, multimem if the fabric has it
        auto *dc = new ncclDevComm();
        ncclDevCommRequirements req = {};
        req.lsaMultimem = true;
        ncclResult_t r = ncclDevCommCreate(ctx->comm, &req, dc);
        if (r != ncclSuccess) {
            req.lsaMultimem = false;
            r = ncclDevCommCreate(ctx->comm, &req, dc);
        }
        ctx->devcomm_state = r == ncclSuccess ? 1 : 0;
        if (ctx->devcomm_state) ctx->devcomm = dc;
        else delete dc;
    }
    if (ctx->devcomm_state == 1) {
        const auto *dc = static_cast<const ncclDevComm *>(ctx->devcomm);
        if (dc->lsaMultimem.mcBasePtr)
            rec.mc = static_cast<char *>(dc->lsaMultimem.mcBasePtr) + (size_t)wv.mcOffset4K * 4096;
    }
    // the window's own slot must be this rank's (the flat mapping gives every
    // rank's buffer a second address, its own included); agreed by all ranks
    TRY(rank_agree(ctx, s, wv.lsaRank == ctx->rank, &all));
    if (!all) {
        ncclCommWindowDeregister(ctx->comm, win);
        if (getenv("SKEL_LOG")) fprintf(stderr, "[skel] NCCL symmetric window: LSA rank mismatch on some rank\n");
        return SKEL_OK;
    }
    ctx->wins[nb] = rec;
    *ok = true;
    if (getenv("SKEL_LOG"))
        fprintf(stderr, "[skel] NCCL symmetric window: rank %d, %zu bytes (ncclMemAlloc + ncclCommWindowRegister), "
                        "%d LSA peers, multicast %s\n",
                ctx->rank, size, ctx->D, rec.mc ? "yes" : "no (device communicator without lsaMultimem)");
    return SKEL_OK;
}

// ---- Reduce / Scan -------------------------------------------------------------
using PFN_encode = CUresult (*)(CUtensorMap *, CUtensorMapDataType, cuuint32_t, void *, const cuuint64_t *,
                                const cuuint64_t *, const cuuint32_t *, const cuuint32_t *, CUtensorMapInterleave,
                                CUtensorMapSwizzle, CUtensorMapL2promotion, CUtensorMapFloatOOBfill);
PFN_encode get_encode() {
    static PFN_encode fn = nullptr;
    static std::once_flag once;
    std::call_once(once, [] {
        void *p = nullptr;
        cudaDriverEntryPointQueryResult q;
        if (cudaGetDriverEntryPointByVersion("cuTensorMapEncodeTiled", &p, 12000, cudaEnableDefault, &q) ==
                cudaSuccess &&
            q == cudaDriverEntryPointSuccess)
            fn = reinterpret_cast<PFN_encode>(p);
    });
    return fn;
}

// 2-D view [rows][128 B] of a tile-aligned prefix, 128B swizzle, 256-row boxes
bool make_tmap(CUtensorMap *map, const void *ptr, uint64_t rows, uint32_t box_rows = 256) {
    memset(map, 0, sizeof *map);
    PFN_encode enc = get_encode();
    if (!enc || rows == 0 || !al16(ptr) || rows > 0x7fffffffull) return false;
    cuuint64_t dims[2] = {32, rows};
    cuuint64_t strides[1] = {128};
    cuuint32_t box[2] = {32, box_rows};
    cuuint32_t estr[2] = {1, 1};
    CUresult r = enc(map, CU_TENSOR_MAP_DATA_TYPE_UINT32, 2, const_cast<void *>(ptr), dims, strides, box, estr,
                     CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_128B, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                     CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    return r == CUDA_SUCCESS;
}

struct RedLayout {  // per-slot workspace carve-up (bytes)
    size_t slot;    // sizeof(slot<T>), padded to 16
    size_t o_res, o_seed, o_gather, o_fold, o_part, o_pvalid, o_aggv, o_incv, total;
};
RedLayout red_layout(const Module *m, int D, size_t G, size_t ntiles) {
    RedLayout L{};
    L.slot = align_up(m->sig[4], 16);
    size_t o = 0;
    L.o_res = o;
    o += L.slot;
    L.o_seed = o;
    o += L.slot;
    L.o_fold = o;
    o += L.slot;
    o = align_up(o, 256);
    L.o_gather = o;
    o = align_up(o + (size_t)D * L.slot, 256);
    L.o_part = o;
    o = align_up(o + G * L.slot, 256);
    L.o_pvalid = o;
    o = align_up(o + G * 4, 256);
    L.o_aggv = o;
    o = align_up(o + (m->sig[13] ? 0 : ntiles * L.slot), 256);
    L.o_incv = o;
    o = align_up(o + (m->sig[13] ? 0 : ntiles * L.slot), 256);
    L.total = o;
    return L;
}
int ensure_ws(skel_ctx_s *ctx, Slot &s, size_t bytes) {
    if (s.ws_cap >= bytes) return SKEL_OK;
    TRY(dev_free(ctx, s, s.ws));
    s.ws = nullptr;
    s.ws_cap = 0;
    const size_t b = std::max<size_t>(bytes, 1 << 20);
    TRY(dev_alloc(ctx, s, b, &s.ws));
    s.ws_cap = b;
    return SKEL_OK;
}
int ensure_status(skel_ctx_s *ctx, Slot &s, size_t ntiles, bool packed) {
    DevGuard g(s.dev);
    if (packed && s.st64_cap < ntiles) {
        TRY(dev_free(ctx, s, reinterpret_cast<char *>(s.st64)));
        char *p = nullptr;
        TRY(dev_alloc(ctx, s, ntiles * 8, &p));
        CK(ctx, cudaMemsetAsync(p, 0, ntiles * 8, s.stream));
        s.st64 = reinterpret_cast<unsigned long long *>(p);
        s.st64_cap = ntiles;
    }
    if (!packed && s.fl32_cap < ntiles) {
        TRY(dev_free(ctx, s, reinterpret_cast<char *>(s.fl32)));
        char *p = nullptr;
        TRY(dev_alloc(ctx, s, ntiles * 4, &p));
        CK(ctx, cudaMemsetAsync(p, 0, ntiles * 4, s.stream));
        s.fl32 = reinterpret_cast<unsigned *>(p);
        s.fl32_cap = ntiles;
    }
    return SKEL_OK;
}
int set_smem_attr(skel_ctx_s *ctx, Module *m, const Slot &s) {
    if (m->attr_set_on.count(s.dev)) return SKEL_OK;
    DevGuard g(s.dev);
    const int dsm = (int)m->sig[11];
    if (dsm > 0) {
        CK(ctx, cudaFuncSetAttribute((const void *)m->k_main, cudaFuncAttributeMaxDynamicSharedMemorySize, dsm));
    }
    if (m->sig[12] > 0) {
        CK(ctx, cudaFuncSetAttribute((const void *)m->k_scan, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                     (int)m->sig[12]));
    }
    m->attr_set_on.insert(s.dev);
    return SKEL_OK;
}

// resident Reduce CTAs per SM (the grid is SMs x this, capped by the tile count)
int red_occupancy(Module *m, const Slot &s) {
    if (m->red_occ > 0) return m->red_occ;
    int occ = 1;
    DevGuard g(s.dev);
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, (const void *)m->k_main, (int)m->sig[9],
                                                      (size_t)m->sig[11]) != cudaSuccess || occ < 1) {
        cudaGetLastError();
        occ = 1;
    }
    if (const char *e = getenv("SKEL_RED_OCC")) occ = std::max(1, std::min(occ, atoi(e)));  // tuning hook
    m->red_occ = occ;
    return occ;
}

// Reduce grid.  Up to ~55 tiles per SM: one CTA per resident slot, static
// contiguous tile ranges.  Larger vectors: oversubscribe (2/4/8 CTAs per slot,
// still contiguous ranges) so the hardware scheduler hands the last ranges to
// whichever SMs finish first -- measured at 2^28/2^29/2^30 floats: 168->161,
// 326->310, 629->605 us; below that the pipeline fill of each extra CTA costs
// more than the balance gains (tools/red_variants.sh).
size_t red_grid(Module *m, const Slot &s, uint64_t cnt) {
    static const int os_env = [] {  // tuning hook SKEL_RED_OVERSUB (CTAs per resident slot)
        const char *e = getenv("SKEL_RED_OVERSUB");
        return e ? std::max(1, atoi(e)) : 0;
    }();
    const uint64_t slots = (uint64_t)s.sms * (uint64_t)red_occupancy(m, s);
    const uint64_t nft = cnt / m->sig[10];
    uint64_t os = os_env;
    if (!os) os = std::min<uint64_t>(8, std::max<uint64_t>(1, nft / (slots * 55)));
    if (os > 2 && os < 8) os = os < 6 ? 4 : 8;  // powers of two (measured points)
    return (size_t)std::max<uint64_t>(1, std::min<uint64_t>(slots * os, nft));
}

// partial results the Reduce kernel publishes: one per CTA, or one per tile
// (+ the ragged tail) in the interleaved tile order (sig[15] bit 48)
size_t red_parts(Module *m, const Slot &s, uint64_t cnt) {
    const size_t G = red_grid(m, s, cnt);
    if (!((m->sig[15] >> 48) & 1)) return G;
    return std::max<size_t>(G, (size_t)(cnt / m->sig[10]) + 1);
}

// small vectors: tile aggregates + a one-CTA ordered fold (two short launches)
// up to SKEL_RED_SMALL_MAX elements (tuning hook; default 128 MiB of elements:
// measured crossover with the TMA kernel between 2^25 and 2^26 floats).  Above
// 8 MiB the tiles are twice as large (16 elements per thread for floats).
bool red_small_big_tiles(const Module *m, uint64_t cnt) { return cnt * m->sig[3] > (8ull << 20); }
uint64_t red_small_tile(const Module *m, uint64_t cnt) {
    return m->sig[9] * ((m->sig[15] >> 50) & 0xff) * (red_small_big_tiles(m, cnt) ? 2 : 1);
}
bool red_small(const Module *m, uint64_t cnt) {
    static const uint64_t env = [] {
        const char *e = getenv("SKEL_RED_SMALL_MAX");
        return e ? (uint64_t)strtoull(e, nullptr, 10) : ~0ull;
    }();
    const uint64_t mx = env != ~0ull ? env : (uint64_t)(128u << 20) / m->sig[3];
    return m->k_fold_aggs && m->k_red_agg2 && red_small_tile(m, cnt) > 0 && cnt <= mx;
}

// local reduce of the slot's data into dst
// host mirror of red.cuh's skel_xdev (the cross-device single-pass Reduce);
// K == 0: a device-local Reduce
struct XDev {
    void *slots = nullptr;
    unsigned *ticket = nullptr;
    void *dst[16] = {};
    void *gat[16] = {};
    int k = 0, K = 0, ndst = 0;
};
constexpr int kXdevMax = 16;
constexpr int kXdevTicket = 48;  // word of Slot::counters (logical device 0) holding the arrivals

int launch_reduce(skel_ctx_s *ctx, Module *m, Slot &s, const void *in, uint64_t cnt, const RedLayout &L,
                  std::vector<unsigned char> &abuf, void *dst, const XDev &xd = XDev()) {
    if (red_small(m, cnt)) {
        const uint64_t ST = red_small_tile(m, cnt);
        uint64_t nt = (cnt + ST - 1) / ST;
        void *aggs = s.ws + L.total;  // room reserved by reduce_core
        int early = 1;
        const bool big = red_small_big_tiles(m, cnt);
        void *pa_s[] = {&in, &cnt, &aggs, &early, abuf.data()};  // skel_scan_agg_kernel
        void *pa_b[] = {&in, &cnt, &aggs, abuf.data()};          // skel_red_agg2_kernel
        void **pa = big ? pa_b : pa_s;
        DevGuard g(s.dev);
        const void *kagg = big ? (const void *)m->k_red_agg2 : (const void *)m->k_scan_agg;
        CK(ctx, cudaLaunchKernel(kagg, dim3((unsigned)nt), dim3((unsigned)m->sig[9]), pa, 0, s.stream));
        const void *caggs = aggs;
        void *pf[] = {&caggs, &nt, &dst, const_cast<XDev *>(&xd), abuf.data()};
        CK(ctx, launch_dependent((const void *)m->k_fold_aggs, dim3(1), dim3((unsigned)m->sig[9]), pf, s.stream));
        ctx->stats.kernel_launches += 2;
        return SKEL_OK;
    }
    const uint64_t TILE = m->sig[10], RB = m->sig[9];
    const uint64_t nft = cnt / TILE;
    const size_t G = red_grid(m, s, cnt);
    CUtensorMap tin;
    memset(&tin, 0, sizeof tin);
    const bool direct = (m->sig[15] >> 49) & 1;  // direct 128-bit loads: `use_tma` = 16-byte aligned
    int use_tma = m->sig[5] && (direct ? al16(in) : make_tmap(&tin, in, nft * RB, (uint32_t)(RB / 2)));
    char *ws = s.ws;
    void *partials = ws + L.o_part, *pvalid = ws + L.o_pvalid, *result = dst;
    unsigned *counter = s.counters + 2;
    void *params[] = {&tin, &in, &cnt, &use_tma, &partials, &pvalid, &counter, &result, const_cast<XDev *>(&xd),
                      abuf.data()};
    DevGuard g(s.dev);
    CK(ctx, launch_dependent((const void *)m->k_main, dim3((unsigned)G), dim3((unsigned)RB), params, s.stream,
                             use_tma ? m->sig[11] : 0));
    ctx->stats.kernel_launches++;
    return SKEL_OK;
}

// Reduce of `in` leaving the result in every local slot's ws[o_fold]
// (cross-device: gather of the D partials + ordered fold), or --
// one local device and `direct` given -- written by the kernel straight to `direct`
int reduce_core(skel_ctx_s *ctx, Module *m, skel_vec_s *in, const skel_arg *args, int nargs,
                std::vector<RedLayout> &Ls, void *direct = nullptr) {
    const int D = ctx->D;
    const bool cross = D > 1 && in->dist == SKEL_BLOCK;
    const size_t es = m->sig[4];
    const size_t ps = part_size(in->n, D);
    const int K = cross ? (int)((in->n + ps - 1) / ps) : 1;  // devices holding data
    // in-process devices that can all reach each other's memory: one pass, the
    // device-order fold done by the last device to finish (red.cuh skel_xdev)
    static const bool xdev_env = [] {
        const char *e = getenv("SKEL_XDEV_REDUCE");  // 0: gather + fold launches instead
        return !(e && atoi(e) == 0);
    }();
    const bool single = cross && !ctx->rank_mode && ctx->peer_all && ctx->peer_atomics && xdev_env && K <= kXdevMax &&
                        ctx->slots.size() <= (size_t)kXdevMax;
    std::vector<unsigned char> abuf;
    Ls.resize(ctx->slots.size());
    for (size_t li = 0; li < ctx->slots.size(); ++li) {  // every workspace before any launch (XDev points across)
        Slot &s = ctx->slots[li];
        const uint64_t cnt = in->bufs[li].count;
        TRY(set_smem_attr(ctx, m, s));  // before the occupancy query in red_grid
        Ls[li] = red_layout(m, D, red_parts(m, s, cnt), 0);
        const size_t extra =
            red_small(m, cnt) ? (size_t)((cnt + red_small_tile(m, cnt) - 1) / red_small_tile(m, cnt)) * Ls[li].slot : 0;
        TRY(ensure_ws(ctx, s, Ls[li].total + extra));
    }
    XDev xd;
    if (single) {
        xd.slots = ctx->slots[0].ws + Ls[0].o_gather;  // room for D packed slots
        xd.ticket = ctx->slots[0].counters + kXdevTicket;
        xd.K = K;
        xd.ndst = (int)ctx->slots.size();
        for (size_t j = 0; j < ctx->slots.size(); ++j) {
            xd.dst[j] = ctx->slots[j].ws + Ls[j].o_fold;
            xd.gat[j] = ctx->slots[j].ws + Ls[j].o_gather;
        }
    }
    for (size_t li = 0; li < ctx->slots.size(); ++li) {
        Slot &s = ctx->slots[li];
        const uint64_t cnt = in->bufs[li].count;
        pack_args(m, args, nargs, li, abuf);
        char *dst = cross ? s.ws + Ls[li].o_res : (direct && D == 1 ? static_cast<char *>(direct) : s.ws + Ls[li].o_fold);
        xd.k = s.d;
        if (cnt) TRY(launch_reduce(ctx, m, s, in->bufs[li].ptr(in->es), cnt, Ls[li], abuf, dst, xd));
    }
    if (single) {
        ctx->stats.xdev_reduces++;
        return join(ctx);  // every device after the last arriver's stores
    }
    if (cross && !ctx->rank_mode) {
        TRY(join(ctx));
        std::vector<const void *> src0(K);
        std::vector<int> sdev(K);
        for (int j = 0; j < K; ++j) src0[j] = ctx->slots[j].ws + Ls[j].o_res, sdev[j] = ctx->slots[j].dev;
        for (size_t li = 0; li < ctx->slots.size(); ++li) {
            Slot &s = ctx->slots[li];
            std::vector<const void *> src = src0;
            TRY(stage_remote(ctx, s, src, sdev, es));
            DevGuard g(s.dev);
            CK(ctx, launch_gather(s.ws + Ls[li].o_gather, src.data(), K, es, s.stream));  // packed slot<T>[K]
            ctx->stats.kernel_launches++;
        }
        TRY(join(ctx));
    } else if (cross) {
        Slot &s = ctx->slots[0];
        DevGuard g(s.dev);
        NK(ctx, ncclAllGather(s.ws + Ls[0].o_res, s.ws + Ls[0].o_gather, es, ncclUint8, ctx->comm, s.stream));
        ctx->stats.nccl_bytes += es * D;
    }
    for (size_t li = 0; li < ctx->slots.size(); ++li) {
        Slot &s = ctx->slots[li];
        const RedLayout &L = Ls[li];
        DevGuard g(s.dev);
        if (cross) {
            pack_args(m, args, nargs, li, abuf);
            const void *vals = s.ws + L.o_gather;
            void *outp = s.ws + L.o_fold;
            int k = K;
            void *params[] = {&vals, &k, &outp, abuf.data()};
            CK(ctx, launch_dependent((const void *)m->k_fold, dim3(1), dim3(32), params, s.stream));
            ctx->stats.kernel_launches++;
        }
    }
    return SKEL_OK;
}

// make every local device's ws[o_fold] hold the Reduce result
int finish_scalar(skel_ctx_s *ctx, skel_vec_s *in, const std::vector<RedLayout> &Ls) {
    const bool cross = ctx->D > 1 && in->dist == SKEL_BLOCK;
    if (cross || ctx->D == 1 || in->dist == SKEL_COPY) return SKEL_OK;
    // SINGLE on several devices: only logical device 0 computed
    if (ctx->rank_mode) {
        Slot &s = ctx->slots[0];
        DevGuard g(s.dev);
        char *p = s.ws + Ls[0].o_fold;
        NK(ctx, ncclBroadcast(p, p, in->es, ncclUint8, 0, ctx->comm, s.stream));
        ctx->stats.nccl_bytes += in->es;
        return SKEL_OK;
    }
    TRY(join(ctx));
    for (size_t li = 1; li < ctx->slots.size(); ++li) {
        Slot &s = ctx->slots[li];
        DevGuard g(s.dev);
        CK(ctx, cudaMemcpyAsync(s.ws + Ls[li].o_fold, ctx->slots[0].ws + Ls[0].o_fold, in->es, cudaMemcpyDefault,
                                s.stream));
    }
    return join(ctx);
}

int check_red(skel_ctx_s *ctx, Module *m, skel_vec_s *in) {
    if (m->sig[3] != in->es)
        return fail(ctx, SKEL_ERR_TYPE, "element size " + std::to_string(in->es) + " != sizeof(T) = " +
                                            std::to_string(m->sig[3]));
    return SKEL_OK;
}

}  // namespace

// =============================================================================
// C-ABI
// =============================================================================
extern "C" {

const char *skel_status_string(int st) {
    switch (st) {
        case SKEL_OK: return "SKEL_OK";
        case SKEL_ERR_ARG: return "SKEL_ERR_ARG";
        case SKEL_ERR_SIZE: return "SKEL_ERR_SIZE";
        case SKEL_ERR_TYPE: return "SKEL_ERR_TYPE";
        case SKEL_ERR_COMPILE: return "SKEL_ERR_COMPILE";
        case SKEL_ERR_CUDA: return "SKEL_ERR_CUDA";
        case SKEL_ERR_NCCL: return "SKEL_ERR_NCCL";
        case SKEL_ERR_OOM: return "SKEL_ERR_OOM";
        case SKEL_ERR_STATE: return "SKEL_ERR_STATE";
        default: return "SKEL_ERR_UNKNOWN";
    }
}

const char *skel_last_error(skel_ctx_t ctx) { return ctx ? ctx->last_error.c_str() : g_last_error.c_str(); }

static int init_slot(skel_ctx_s *ctx, int d, int dev) {
    Slot s;
    s.d = d;
    s.dev = dev;
    DevGuard g(dev);
    CK(ctx, cudaDeviceGetAttribute(&s.sms, cudaDevAttrMultiProcessorCount, dev));
    {
        int maj = 0, mnr = 0;
        CK(ctx, cudaDeviceGetAttribute(&maj, cudaDevAttrComputeCapabilityMajor, dev));
        CK(ctx, cudaDeviceGetAttribute(&mnr, cudaDevAttrComputeCapabilityMinor, dev));
        s.cc = maj * 10 + mnr;
    }
    CK(ctx, cudaStreamCreateWithFlags(&s.stream, cudaStreamNonBlocking));
    CK(ctx, cudaEventCreateWithFlags(&s.ev, cudaEventDisableTiming));
    CK(ctx, cudaEventCreateWithFlags(&s.ev_scan, cudaEventDisableTiming));
    CK(ctx, cudaStreamCreateWithFlags(&s.dl_stream, cudaStreamNonBlocking));
    CK(ctx, cudaEventCreateWithFlags(&s.dl_ready, cudaEventDisableTiming));
    void *p = nullptr;
    CK(ctx, cudaMalloc(&p, 256));
    CK(ctx, cudaMemsetAsync(p, 0, 256, s.stream));  // ordered with the epoch write below
    s.counters = static_cast<unsigned *>(p);
    const unsigned first_epoch = 1;  // status words are zeroed: epoch 0 must never be live
    CK(ctx, cudaMemcpyAsync(s.counters + 3, &first_epoch, sizeof first_epoch, cudaMemcpyHostToDevice, s.stream));
    CK(ctx, cudaStreamSynchronize(s.stream));
    ctx->slots.push_back(s);
    return SKEL_OK;
}

static void ctx_defaults(skel_ctx_s *ctx) {
    const char *f = getenv("SKEL_FMAD");
    ctx->fmad = f && atoi(f) != 0;
    if (const char *e = getenv("SKEL_VMM")) ctx->vmm_on = atoi(e) != 0;  // 0: cudaMalloc only
    if (const char *e = getenv("SKEL_NCCL_WINDOWS")) ctx->nccl_windows = atoi(e) != 0;
    if (const char *e = getenv("SKEL_VMM_MIN")) ctx->vmm_min = (size_t)strtoull(e, nullptr, 10);
    const char *b = getenv("SKEL_BLOCK_SIZE");
    if (b) ctx->block_size = atoi(b);
}

int skel_init(int num_devices, skel_ctx_t *out) {
    if (!out) return fail(nullptr, SKEL_ERR_ARG, "out is NULL");
    int ngpu = 0;
    cudaError_t e = cudaGetDeviceCount(&ngpu);
    if (e != cudaSuccess || ngpu == 0) {
        cudaGetLastError();
        return fail(nullptr, SKEL_ERR_CUDA,
                    std::string("no CUDA device: ") + (e != cudaSuccess ? cudaGetErrorString(e) : "0 devices"));
    }
    const int D = num_devices < 0 ? ngpu : num_devices;
    if (D < 1 || D > 64) return fail(nullptr, SKEL_ERR_ARG, "num_devices must be -1 or 1..64");
    auto *ctx = new skel_ctx_s();
    ctx_defaults(ctx);
    ctx->D = D;
    for (int d = 0; d < D; ++d) {
        int st = init_slot(ctx, d, d % ngpu);
        if (st != SKEL_OK) {
            g_last_error = ctx->last_error;
            delete ctx;
            return st;
        }
    }
    // peer access between distinct physical devices (NVLink / NVSwitch)
    for (auto &a : ctx->slots)
        for (auto &b : ctx->slots)
            if (a.dev != b.dev) {
                int can = 0;
                cudaDeviceCanAccessPeer(&can, a.dev, b.dev);
                if (can) {
                    int atom = 0;
                    if (cudaDeviceGetP2PAttribute(&atom, cudaDevP2PAttrNativeAtomicSupported, a.dev, b.dev) !=
                            cudaSuccess || !atom) {
                        cudaGetLastError();
                        ctx->peer_atomics = false;
                    }
                    DevGuard g(a.dev);
                    cudaError_t pe = cudaDeviceEnablePeerAccess(b.dev, 0);
                    if (pe == cudaErrorPeerAccessAlreadyEnabled) pe = cudaSuccess;
                    if (pe != cudaSuccess) {
                        cudaGetLastError();
                        ctx->peer_all = false;
                    }
                } else {
                    ctx->peer_all = false;
                }
            }
    *out = ctx;
    return SKEL_OK;
}

int skel_get_unique_id(void *id) {
    if (!id) return fail(nullptr, SKEL_ERR_ARG, "id is NULL");
    ncclUniqueId u;
    ncclResult_t r = ncclGetUniqueId(&u);
    if (r != ncclSuccess) return fail(nullptr, SKEL_ERR_NCCL, ncclGetErrorString(r));
    static_assert(sizeof(u) == 128, "ncclUniqueId is 128 bytes");
    memcpy(id, &u, sizeof u);
    return SKEL_OK;
}

int skel_init_rank(int rank, int world, int cuda_device, const void *id, skel_ctx_t *out) {
    if (!out || world < 1 || rank < 0 || rank >= world) return fail(nullptr, SKEL_ERR_ARG, "bad rank/world");
    if (world > 1 && !id) return fail(nullptr, SKEL_ERR_ARG, "nccl id required for world > 1");
    int ngpu = 0;
    cudaError_t e = cudaGetDeviceCount(&ngpu);
    if (e != cudaSuccess || ngpu == 0 || cuda_device < 0 || cuda_device >= ngpu) {
        cudaGetLastError();
        return fail(nullptr, SKEL_ERR_CUDA, "no such CUDA device");
    }
    auto *ctx = new skel_ctx_s();
    ctx_defaults(ctx);
    ctx->D = world;
    ctx->rank_mode = true;
    ctx->rank = rank;
    int st = init_slot(ctx, rank, cuda_device);
    if (st == SKEL_OK) {  // a one-rank communicator too (the fused tail's rank path uses it)
        ncclUniqueId u;
        memcpy(&u, id, sizeof u);
        DevGuard g(cuda_device);
        ncclResult_t r = ncclCommInitRank(&ctx->comm, world, u, rank);
        if (r != ncclSuccess) st = fail(ctx, SKEL_ERR_NCCL, std::string("ncclCommInitRank: ") + ncclGetErrorString(r));
    }
    if (st != SKEL_OK) {
        g_last_error = ctx->last_error;
        delete ctx;
        return st;
    }
    *out = ctx;
    return SKEL_OK;
}

int skel_vector_destroy(skel_vec_t v);

int skel_finalize(skel_ctx_t ctx) {
    if (!ctx) return fail(nullptr, SKEL_ERR_ARG, "ctx is NULL");
    sync_all(ctx);
    sync_downloads(ctx);
    std::vector<skel_vec_s *> vs(ctx->vecs.begin(), ctx->vecs.end());
    for (auto *v : vs) skel_vector_destroy(v);
    for (auto &kv : ctx->modules) {
        if (kv.second->lib) cudaLibraryUnload(kv.second->lib);
    }
    if (ctx->devcomm) {
        ncclDevCommDestroy(ctx->comm, static_cast<const ncclDevComm *>(ctx->devcomm));
        delete static_cast<ncclDevComm *>(ctx->devcomm);
        ctx->devcomm = nullptr;
    }
    if (ctx->comm) ncclCommDestroy(ctx->comm);
    for (auto &s : ctx->slots) {
        DevGuard g(s.dev);
        cudaFree(s.ws);
        cudaFree(s.scratch);
        cudaFree(s.counters);
        cudaFree(s.st64);
        cudaFree(s.fl32);
        cudaEventDestroy(s.ev);
        cudaEventDestroy(s.ev_scan);
        cudaEventDestroy(s.dl_ready);
        cudaStreamDestroy(s.dl_stream);
        cudaStreamDestroy(s.stream);
    }
    delete ctx;
    return SKEL_OK;
}

int skel_num_devices(skel_ctx_t ctx, int *D, int *L) {
    if (!ctx) return fail(nullptr, SKEL_ERR_ARG, "ctx is NULL");
    if (D) *D = ctx->D;
    if (L) *L = (int)ctx->slots.size();
    return SKEL_OK;
}

int skel_get_stream(skel_ctx_t ctx, int li, void **stream) {
    if (!ctx || !stream || li < 0 || li >= (int)ctx->slots.size()) return fail(ctx, SKEL_ERR_ARG, "bad local index");
    *stream = ctx->slots[li].stream;
    return SKEL_OK;
}

int skel_set_block_size(skel_ctx_t ctx, int threads) {
    if (!ctx) return fail(nullptr, SKEL_ERR_ARG, "ctx is NULL");
    if (threads != 0 && (threads < 32 || threads > 1024 || threads % 32))
        return fail(ctx, SKEL_ERR_ARG, "block size must be 0 or a multiple of 32 in [32, 1024]");
    ctx->block_size = threads;
    return SKEL_OK;
}

int skel_set_cache_dir(skel_ctx_t ctx, const char *dir) {
    if (!ctx) return fail(nullptr, SKEL_ERR_ARG, "ctx is NULL");
    if (!dir) {
        ctx->cache_dir.clear();
        ctx->disk_cache = true;
    } else if (!*dir) {
        ctx->disk_cache = false;
    } else {
        ctx->cache_dir = dir;
        ctx->disk_cache = true;
    }
    return SKEL_OK;
}

int skel_clear_kernel_cache(skel_ctx_t ctx) {
    if (!ctx) return fail(nullptr, SKEL_ERR_ARG, "ctx is NULL");
    TRY(sync_all(ctx));
    for (auto &kv : ctx->modules) {
        if (kv.second->lib) cudaLibraryUnload(kv.second->lib);
    }
    ctx->modules.clear();
    ctx->fast_modules.clear();
    return SKEL_OK;
}

int skel_sync(skel_ctx_t ctx) {
    SKEL_RANGE("skel_sync");
    if (!ctx) return fail(nullptr, SKEL_ERR_ARG, "ctx is NULL");
    TRY(sync_all(ctx));
    return sync_downloads(ctx);
}

int skel_get_stats(skel_ctx_t ctx, skel_stats *out) {
    if (!ctx || !out) return fail(ctx, SKEL_ERR_ARG, "NULL argument");
    *out = ctx->stats;
    return SKEL_OK;
}

int skel_reset_stats(skel_ctx_t ctx) {
    if (!ctx) return fail(nullptr, SKEL_ERR_ARG, "ctx is NULL");
    ctx->stats = skel_stats{};
    return SKEL_OK;
}

// ---- vectors -------------------------------------------------------------------
int skel_vector_create(skel_ctx_t ctx, size_t n, size_t es, skel_vec_t *out) {
    if (!ctx || !out || es == 0) return fail(ctx, SKEL_ERR_ARG, "bad vector arguments");
    auto *v = new skel_vec_s();
    v->ctx = ctx;
    v->serial = ++ctx->next_serial;
    v->n = n;
    v->es = es;
    v->dist = ctx->D == 1 ? SKEL_SINGLE : SKEL_BLOCK;
    v->bufs.resize(ctx->slots.size());
    int st = place(v, v->dist);
    for (size_t li = 0; st == SKEL_OK && li < ctx->slots.size(); ++li) {
        Slot &s = ctx->slots[li];
        Buf &b = v->bufs[li];
        DevGuard g(s.dev);
        if (b.cap) {
            cudaError_t e = cudaMemsetAsync(b.base, 0, b.cap, s.stream);
            if (e != cudaSuccess) st = fail(ctx, SKEL_ERR_CUDA, cudaGetErrorString(e));
        }
    }
    if (st != SKEL_OK) {
        for (size_t li = 0; li < v->bufs.size(); ++li) dev_free(ctx, ctx->slots[li], v->bufs[li].base);
        delete v;
        return st;
    }
    v->dev_valid = true;
    v->host_valid = false;
    ctx->vecs.insert(v);
    *out = v;
    return SKEL_OK;
}

int skel_vector_destroy(skel_vec_t v) {
    if (!v) return fail(nullptr, SKEL_ERR_ARG, "vector is NULL");
    skel_ctx_s *ctx = v->ctx;
    mc_release(v);
    for (auto &b : v->bufs) close_peers(b);
    for (size_t li = 0; li < v->bufs.size(); ++li) dev_free(ctx, ctx->slots[li], v->bufs[li].base);
    for (size_t li = 0; li < v->bufs.size(); ++li)
        if (v->bufs[li].dl_done) {
            DevGuard g(ctx->slots[li].dev);
            cudaEventDestroy(v->bufs[li].dl_done);
        }
    if (v->host) cudaFreeHost(v->host);
    ctx->vecs.erase(v);
    delete v;
    return SKEL_OK;
}

int skel_vector_set_dtype(skel_vec_t v, skel_dtype dt) {
    if (!v) return fail(nullptr, SKEL_ERR_ARG, "vector is NULL");
    static const size_t sz[] = {0, 4, 8, 4, 4, 8, 8};
    if ((int)dt < 0 || (int)dt > 6) return fail(v->ctx, SKEL_ERR_ARG, "bad dtype");
    if (dt != SKEL_DT_OPAQUE && sz[dt] != v->es) return fail(v->ctx, SKEL_ERR_TYPE, "dtype size != elem_size");
    v->dt = dt;
    return SKEL_OK;
}

int skel_vector_size(skel_vec_t v, size_t *n, size_t *es) {
    if (!v) return fail(nullptr, SKEL_ERR_ARG, "vector is NULL");
    if (n) *n = v->n;
    if (es) *es = v->es;
    return SKEL_OK;
}

int skel_vector_upload(skel_vec_t v, const void *src, size_t n) {
    SKEL_RANGE("skel_vector_upload");
    if (!v || (!src && n)) return fail(v ? v->ctx : nullptr, SKEL_ERR_ARG, "bad upload arguments");
    if (n != v->n) return fail(v->ctx, SKEL_ERR_SIZE, "upload length != vector length");
    TRY(host_mirror(v));  // (replaces a rank-local part mirror)
    // the host mirror may still be the source of an in-flight H2D copy
    TRY(sync_all(v->ctx));
    if (n) memcpy(v->host, src, n * v->es);
    v->host_valid = true;
    v->dev_valid = false;  // H2D deferred until a skeleton needs the data
    v->diverged = false;
    return SKEL_OK;
}

int skel_vector_upload_part(skel_vec_t v, size_t lo, const void *src, size_t count) {
    SKEL_RANGE("skel_vector_upload_part");
    if (!v || (!src && count)) return fail(v ? v->ctx : nullptr, SKEL_ERR_ARG, "bad upload_part arguments");
    skel_ctx_s *ctx = v->ctx;
    if (lo > v->n || count > v->n - lo) return fail(ctx, SKEL_ERR_SIZE, "range outside the vector");
    size_t plo = 0, phi = 0;
    if (ctx->rank_mode && v->dist == SKEL_BLOCK) part_range(v->n, ctx->D, ctx->rank, &plo, &phi);
    TRY(sync_all(ctx));  // the mirror may still feed an in-flight H2D
    if (ctx->rank_mode && ctx->D > 1 && v->dist == SKEL_BLOCK && lo == plo && count == phi - plo &&
        !(v->host && !partial_mirror(v) && v->host_valid)) {
        // this process's part only: a rank-local mirror (no full-size host copy)
        if (!partial_mirror(v) || v->host_lo != plo) {
            if (v->host) cudaFreeHost(v->host);
            v->host = nullptr;
            void *p = nullptr;
            cudaError_t e = cudaHostAlloc(&p, std::max<size_t>(count * v->es, 16), cudaHostAllocPortable);
            if (e != cudaSuccess) {
                cudaGetLastError();
                return fail(ctx, SKEL_ERR_OOM, std::string("cudaHostAlloc: ") + cudaGetErrorString(e));
            }
            v->host = static_cast<char *>(p);
            v->host_lo = plo;
            v->host_n = count;
        }
        if (count) memcpy(v->host, src, count * v->es);
    } else {
        if (lo == 0 && count == v->n) TRY(host_mirror(v));
        else if (!v->host_valid) TRY(ensure_host(v));  // the rest of the host copy must be current
        if (count) memcpy(v->host + lo * v->es, src, count * v->es);
    }
    v->host_valid = true;
    v->dev_valid = false;
    v->diverged = false;
    return SKEL_OK;
}

int skel_vector_download(skel_vec_t v, void *dst, size_t n) {
    SKEL_RANGE("skel_vector_download");
    if (!v || (!dst && n)) return fail(v ? v->ctx : nullptr, SKEL_ERR_ARG, "bad download arguments");
    if (n != v->n) return fail(v->ctx, SKEL_ERR_SIZE, "download length != vector length");
    if (partial_mirror(v)) {
        // rank-local host data: assemble the whole vector on the devices, then read it
        TRY(ensure_device(v));
        v->host_valid = false;
        cudaFreeHost(v->host);
        v->host = nullptr;
    }
    TRY(ensure_host(v));
    if (n) memcpy(dst, v->host, n * v->es);
    return SKEL_OK;
}

namespace {
int download_range(skel_vec_s *v, size_t lo, void *dst, size_t count, bool async);
}
int skel_vector_download_part(skel_vec_t v, size_t lo, void *dst, size_t count) {
    SKEL_RANGE("skel_vector_download_part");
    return download_range(v, lo, dst, count, false);
}
int skel_vector_download_part_async(skel_vec_t v, size_t lo, void *dst, size_t count) {
    SKEL_RANGE("skel_vector_download_part_async");
    return download_range(v, lo, dst, count, true);
}
namespace {
int download_range(skel_vec_s *v, size_t lo, void *dst, size_t count, bool async) {
    if (!v || (!dst && count)) return fail(v ? v->ctx : nullptr, SKEL_ERR_ARG, "bad download_part arguments");
    if (v->ctx->capturing)
        return fail(v->ctx, SKEL_ERR_STATE, "downloads cannot be captured into a graph (skel_capture_begin)");
    skel_ctx_s *ctx = v->ctx;
    if (lo > v->n || count > v->n - lo) return fail(ctx, SKEL_ERR_SIZE, "range outside the vector");
    if (!count) return SKEL_OK;
    const size_t es = v->es, hi = lo + count;
    if (v->host_valid && v->host && lo >= v->host_lo && hi <= v->host_lo + v->host_n) {
        TRY(sync_all(ctx));  // the mirror may still be the target of an in-flight D2H
        memcpy(dst, v->host + (lo - v->host_lo) * es, count * es);
        return SKEL_OK;
    }
    if (!v->dev_valid) TRY(ensure_device(v));
    // which local slots hold [lo, hi) and where
    struct Piece { size_t li, src_off, lo, cnt; };
    std::vector<Piece> pieces;
    bool covered = false;
    if (v->dist == SKEL_BLOCK && ctx->D > 1) {
        size_t got = 0;
        for (size_t li = 0; li < ctx->slots.size(); ++li) {
            size_t plo, phi;
            part_range(v->n, ctx->D, ctx->slots[li].d, &plo, &phi);
            const size_t a = std::max(lo, plo), b = std::min(hi, phi);
            if (a < b) {
                pieces.push_back({li, a - plo, a, b - a});
                got += b - a;
            }
        }
        covered = got == count;
    } else if (v->dist == SKEL_COPY || ctx->D == 1) {
        // device 0's copy (reading R6) -- or, in rank mode, the local copy if it cannot have diverged
        if (!ctx->rank_mode || ctx->D == 1 || !v->diverged) {
            pieces.push_back({0, lo, lo, count});
            covered = true;
        }
    } else if (v->dist == SKEL_SINGLE && ctx->slots[0].d == 0) {
        pieces.push_back({0, lo, lo, count});
        covered = true;
    }
    if (!covered && ctx->rank_mode)  // a collective fallback would need every rank to take it
        return fail(ctx, SKEL_ERR_STATE, "download_part in rank mode: the range is not held by this rank");
    if (!covered) {  // in-process devices: the full download
        TRY(ensure_host(v));
        memcpy(dst, v->host + lo * es, count * es);
        return SKEL_OK;
    }
    for (const Piece &p : pieces) {
        Slot &s = ctx->slots[p.li];
        Buf &b = v->bufs[p.li];
        DevGuard g(s.dev);
        char *to = static_cast<char *>(dst) + (p.lo - lo) * es;
        const char *from = b.ptr(es) + p.src_off * es;
        if (async) {  // on the download stream, after everything enqueued on the main stream so far
            CK(ctx, cudaEventRecord(s.dl_ready, s.stream));
            CK(ctx, cudaStreamWaitEvent(s.dl_stream, s.dl_ready, 0));
            CK(ctx, cudaMemcpyAsync(to, from, p.cnt * es, cudaMemcpyDeviceToHost, s.dl_stream));
            if (!b.dl_done) CK(ctx, cudaEventCreateWithFlags(&b.dl_done, cudaEventDisableTiming));
            CK(ctx, cudaEventRecord(b.dl_done, s.dl_stream));
            b.dl_pending = true;
        } else {
            CK(ctx, cudaMemcpyAsync(to, from, p.cnt * es, cudaMemcpyDeviceToHost, s.stream));
        }
        ctx->stats.d2h_bytes += p.cnt * es;
        ctx->stats.d2h_copies++;
    }
    return async ? SKEL_OK : sync_all(ctx);
}
}  // namespace

int skel_vector_host_ptr(skel_vec_t v, void **host) {
    SKEL_RANGE("skel_vector_host_ptr");
    if (!v || !host) return fail(v ? v->ctx : nullptr, SKEL_ERR_ARG, "bad arguments");
    TRY(ensure_host(v));
    *host = v->host;
    return SKEL_OK;
}

int skel_vector_mark_host_modified(skel_vec_t v) {
    if (!v) return fail(nullptr, SKEL_ERR_ARG, "vector is NULL");
    if (!v->host) return fail(v->ctx, SKEL_ERR_STATE, "vector has no host mirror (call skel_vector_host_ptr)");
    v->host_valid = true;
    v->dev_valid = false;
    v->diverged = false;
    return SKEL_OK;
}

int skel_vector_fill(skel_vec_t v, const void *value) {
    if (!v) return fail(nullptr, SKEL_ERR_ARG, "vector is NULL");
    return skel_vector_fill_dist(v, v->dist, value);
}

int skel_vector_fill_dist(skel_vec_t v, skel_dist dist, const void *value) {
    SKEL_RANGE("skel_vector_fill_dist");
    if (!v || !value || (int)dist < 0 || (int)dist > 2)
        return fail(v ? v->ctx : nullptr, SKEL_ERR_ARG, "bad fill arguments");
    skel_ctx_s *ctx = v->ctx;
    TRY(wait_dl(v));
    v->dist = dist;  // old contents are discarded: no exchange needed
    if (v->es > 64) return fail(ctx, SKEL_ERR_TYPE, "fill supports elements up to 64 bytes");
    TRY(place(v, v->dist));
    for (size_t li = 0; li < ctx->slots.size(); ++li) {
        Slot &s = ctx->slots[li];
        Buf &b = v->bufs[li];
        if (!b.count) continue;
        DevGuard g(s.dev);
        CK(ctx, launch_fill(b.ptr(v->es), b.count, value, v->es, s.stream));
        ctx->stats.kernel_launches++;
    }
    v->dev_valid = true;
    device_wrote(v);
    v->diverged = false;
    return SKEL_OK;
}

int skel_vector_set_distribution(skel_vec_t v, skel_dist dist, skel_combine combine) {
    SKEL_RANGE("skel_vector_set_distribution");
    if (!v) return fail(nullptr, SKEL_ERR_ARG, "vector is NULL");
    if ((int)dist < 0 || (int)dist > 2 || (int)combine < 0 || (int)combine > 4)
        return fail(v->ctx, SKEL_ERR_ARG, "bad distribution or combine");
    return set_distribution(v, dist, combine);
}

int skel_vector_set_distribution_fn(skel_vec_t v, skel_dist dist, const char *combine_src) {
    SKEL_RANGE("skel_vector_set_distribution_fn");
    if (!v || !combine_src) return fail(v ? v->ctx : nullptr, SKEL_ERR_ARG, "bad arguments");
    if ((int)dist < 0 || (int)dist > 2) return fail(v->ctx, SKEL_ERR_ARG, "bad distribution");
    return set_distribution_fn(v, dist, combine_src);
}

int skel_vector_get_distribution(skel_vec_t v, skel_dist *dist) {
    if (!v || !dist) return fail(v ? v->ctx : nullptr, SKEL_ERR_ARG, "bad arguments");
    *dist = v->dist;
    return SKEL_OK;
}

int skel_vector_mark_device_modified(skel_vec_t v) {
    SKEL_RANGE("skel_vector_mark_device_modified");
    if (!v) return fail(nullptr, SKEL_ERR_ARG, "vector is NULL");
    TRY(ensure_device(v));
    device_wrote(v);
    if (v->dist == SKEL_COPY && v->ctx->D > 1) v->diverged = true;
    return SKEL_OK;
}

int skel_vector_part(skel_vec_t v, int d, size_t *lo, size_t *hi) {
    if (!v || !lo || !hi || d < 0 || d >= v->ctx->D) return fail(v ? v->ctx : nullptr, SKEL_ERR_ARG, "bad arguments");
    if (v->dist == SKEL_BLOCK) {
        part_range(v->n, v->ctx->D, d, lo, hi);
    } else if (v->dist == SKEL_COPY || d == 0) {
        *lo = 0;
        *hi = v->n;
    } else {
        *lo = *hi = 0;
    }
    return SKEL_OK;
}

int skel_vector_device_ptr(skel_vec_t v, int li, void **ptr, size_t *count) {
    if (!v || li < 0 || li >= (int)v->bufs.size()) return fail(v ? v->ctx : nullptr, SKEL_ERR_ARG, "bad arguments");
    TRY(ensure_device(v));
    if (ptr) *ptr = v->bufs[li].ptr(v->es);
    if (count) *count = v->bufs[li].count;
    return SKEL_OK;
}

// ---- skeletons -------------------------------------------------------------------
int skel_map(skel_ctx_t ctx, const char *src, skel_vec_t in, skel_vec_t out, const skel_arg *args, int nargs) {
    SKEL_RANGE("skel_map");
    if (!ctx || !src || !in || in->ctx != ctx || (out && out->ctx != ctx) || (nargs && !args) || nargs < 0)
        return fail(ctx, SKEL_ERR_ARG, "bad map arguments");
    return run_ew(ctx, Kind::Map, src, in, nullptr, out, args, nargs);
}

// index Map: out[i] = f(i, args...) for i in [0, n) without an
// input vector; each device computes the indices of its part of out (block: its
// part, copy: all, single: device 0); a void f runs over a block partition of [0, n)
int skel_map_index(skel_ctx_t ctx, const char *src, size_t n, skel_vec_t out, const skel_arg *args, int nargs) {
    SKEL_RANGE("skel_map_index");
    if (!ctx || !src || (out && out->ctx != ctx) || (nargs && !args) || nargs < 0)
        return fail(ctx, SKEL_ERR_ARG, "bad map_index arguments");
    Module *m = nullptr;
    TRY(get_module(ctx, Kind::Idx, src, &m));
    const uint64_t rsz = m->sig[3];
    if (rsz != 0 && !out) return fail(ctx, SKEL_ERR_ARG, "non-void function needs an output vector");
    if (rsz != 0 && out->es != rsz)
        return fail(ctx, SKEL_ERR_TYPE, "output element size " + std::to_string(out->es) + " != sizeof(result) = " +
                                            std::to_string(rsz));
    if (m->sig[4] < 8 && n > 0x7fffffffull)
        return fail(ctx, SKEL_ERR_SIZE, "index range exceeds a 4-byte index parameter");
    TRY(check_args(ctx, m, args, nargs));
    skel_dist dist = ctx->D == 1 ? SKEL_SINGLE : SKEL_BLOCK;
    if (rsz != 0) {
        dist = out->dist;
        TRY(prepare_output(out, n, dist, false));
    }
    const int block = (int)m->sig[9];
    const uint64_t E = m->sig[8];
    std::vector<unsigned char> abuf;
    for (size_t li = 0; li < ctx->slots.size(); ++li) {
        Slot &s = ctx->slots[li];
        uint64_t cnt, base;
        void *po = nullptr;
        if (rsz != 0) {
            cnt = out->bufs[li].count;
            base = dist == SKEL_BLOCK ? part_lo(out, s.d) : 0;
            po = out->bufs[li].ptr(out->es);
        } else {
            size_t lo, hi;
            part_range(n, ctx->D, s.d, &lo, &hi);
            cnt = hi - lo;
            base = lo;
        }
        if (!cnt) continue;
        int vec_ok = !po || al16(po);
        pack_args(m, args, nargs, li, abuf);
        const size_t chunks = vec_ok && rsz != 0 ? std::max<uint64_t>(cnt / E, 1) : cnt;
        DevGuard g(s.dev);
        // measured choice between one chunk of E outputs per thread (policy 1) and
        // one element per thread through the scalar path (policy 2): a divergent,
        // compute-bound function (Mandelbrot) balances better with the second
        int policy = 1;
        if (vec_ok && rsz != 0 && E > 1)
            TRY(ew_decide(ctx, m, s, Kind::Idx, nullptr, 0, nullptr, 0, rsz, cnt, base, abuf, 0x26u, &policy));
        // (policy 5: the scalar path over half a grid, two indices per thread)
        const bool scalar = policy == 2 || policy == 5;
        int vk = scalar ? 0 : vec_ok;
        const int grid = ew_grid(s, scalar ? cnt : chunks, block, policy == 5 ? 2 : 1);
        void *params[] = {&po, &cnt, &base, &vk, abuf.data()};
        CK(ctx, launch_dependent((const void *)m->k_main, dim3(grid), dim3(block), params, s.stream));
        ctx->stats.kernel_launches++;
    }
    if (rsz != 0) {
        out->dev_valid = true;
        device_wrote(out);
    }
    return SKEL_OK;
}

// lanes Map: `lanes` threads per element (see map.cuh, SKEL_LANES)
int skel_map_lanes(skel_ctx_t ctx, const char *src, skel_vec_t in, skel_vec_t out, int lanes, const skel_arg *args,
                   int nargs) {
    SKEL_RANGE("skel_map_lanes");
    if (!ctx || !src || !in || in->ctx != ctx || (out && out->ctx != ctx) || (nargs && !args) || nargs < 0)
        return fail(ctx, SKEL_ERR_ARG, "bad map_lanes arguments");
    if (lanes < 1 || lanes > 32 || (lanes & (lanes - 1)))
        return fail(ctx, SKEL_ERR_ARG, "lanes must be a power of two in [1, 32]");
    Module *m = nullptr;
    TRY(get_module(ctx, Kind::Lanes, src, &m));
    const uint64_t rsz = m->sig[3];
    if (m->sig[4] != in->es)
        return fail(ctx, SKEL_ERR_TYPE, "element size " + std::to_string(in->es) + " != sizeof(parameter 0) = " +
                                            std::to_string(m->sig[4]));
    if (rsz != 0 && !out) return fail(ctx, SKEL_ERR_ARG, "non-void function needs an output vector");
    if (rsz != 0 && out->es != rsz)
        return fail(ctx, SKEL_ERR_TYPE, "output element size " + std::to_string(out->es) + " != sizeof(result) = " +
                                            std::to_string(rsz));
    TRY(check_args(ctx, m, args, nargs));
    TRY(ensure_device(in));
    if (rsz != 0) TRY(prepare_output(out, in->n, in->dist, out == in));
    const int block = (int)m->sig[9];
    std::vector<unsigned char> abuf;
    for (size_t li = 0; li < ctx->slots.size(); ++li) {
        Slot &s = ctx->slots[li];
        uint64_t cnt = in->bufs[li].count;
        if (!cnt) continue;
        const void *pa = in->bufs[li].ptr(in->es);
        const void *pb = nullptr;
        void *po = (rsz != 0) ? out->bufs[li].ptr(out->es) : nullptr;
        pack_args(m, args, nargs, li, abuf);
        // one thread per (element, lane): whole warps, up to the grid cap
        const uint64_t threads = (cnt + 32 / lanes - 1) / (32 / lanes) * 32;
        const int grid = ew_grid(s, (size_t)threads, block, 1);
        int ln = lanes;
        void *params[] = {&pa, &pb, &po, &cnt, &ln, abuf.data()};
        DevGuard g(s.dev);
        CK(ctx, launch_dependent((const void *)m->k_main, dim3(grid), dim3(block), params, s.stream));
        ctx->stats.kernel_launches++;
    }
    if (rsz != 0) {
        out->dev_valid = true;
        device_wrote(out);
    }
    return SKEL_OK;
}

int skel_zip(skel_ctx_t ctx, const char *src, skel_vec_t a, skel_vec_t b, skel_vec_t out, const skel_arg *args,
             int nargs) {
    SKEL_RANGE("skel_zip");
    if (!ctx || !src || !a || !b || !out || a->ctx != ctx || b->ctx != ctx || out->ctx != ctx || (nargs && !args) ||
        nargs < 0)
        return fail(ctx, SKEL_ERR_ARG, "bad zip arguments");
    if (a->n != b->n) return fail(ctx, SKEL_ERR_SIZE, "zip: vectors of unequal length (P:L268-269)");
    return run_ew(ctx, Kind::Zip, src, a, b, out, args, nargs);
}

int skel_zip_combine(skel_ctx_t ctx, const char *src, skel_vec_t a, skel_vec_t b, skel_combine combine,
                     skel_vec_t out, const skel_arg *args, int nargs) {
    SKEL_RANGE("skel_zip_combine");
    if (!ctx || !src || !a || !b || !out || a->ctx != ctx || b->ctx != ctx || out->ctx != ctx || (nargs && !args) ||
        nargs < 0 || (int)combine < 1 || (int)combine > 4 || out == b)
        return fail(ctx, SKEL_ERR_ARG, "bad zip_combine arguments");
    if (a->n != b->n) return fail(ctx, SKEL_ERR_SIZE, "zip: vectors of unequal length (P:L268-269)");
    if (b->dt == SKEL_DT_OPAQUE) return fail(ctx, SKEL_ERR_TYPE, "combine needs a numeric dtype (skel_vector_set_dtype)");
    if (b->dist != SKEL_COPY && ctx->D > 1)
        return fail(ctx, SKEL_ERR_STATE, "a combine merges per-device copies: b must be SKEL_COPY");
    const int D = ctx->D;
    // in-process mode loads and stores through the other devices' buffers: only
    // with peer access between every pair of distinct GPUs (else the unfused
    // reduce-scatter + Zip + all-gather, which moves data with copies)
    // SKEL_FORCE_MULTIMEM=1 (test hook): a one-device context takes the fused
    // multicast path too (a multicast object of one device), so the NVLS
    // kernel and the binding can be exercised on a single GPU -- in rank mode a
    // one-rank communicator's fused tail (with SKEL_NCCL_WINDOWS=1: real NCCL
    // symmetric memory on the one GPU a test box has)
    static const bool force_mm = getenv("SKEL_FORCE_MULTIMEM") && atoi(getenv("SKEL_FORCE_MULTIMEM")) != 0;
    const bool fused = ((D > 1 && D <= 16) || (force_mm && D == 1)) &&
                       (a->dist == SKEL_COPY || a->dist == SKEL_BLOCK || D == 1) &&
                       (out != a || a->dist == SKEL_COPY || D == 1) && !ctx->capturing &&
                       (ctx->rank_mode || ctx->peer_all);
    auto unfused = [&]() -> int {  // the same result as the fused kernel
        if (D > 1) TRY(set_distribution(b, SKEL_BLOCK, combine));
        if (a->dist != b->dist) TRY(set_distribution(a, b->dist, SKEL_COMBINE_NONE));
        TRY(run_ew(ctx, Kind::Zip, src, a, b, out, args, nargs));
        return D > 1 ? set_distribution(out, SKEL_COPY, SKEL_COMBINE_NONE) : SKEL_OK;
    };
    if (!fused) return unfused();
    Module *m = nullptr;
    TRY(get_module(ctx, Kind::Zip, src, &m));
    if (m->sig[4] != a->es || m->sig[5] != b->es)
        return fail(ctx, SKEL_ERR_TYPE, "element sizes do not match the zip function's parameters");
    if (m->sig[3] == 0 || m->sig[3] != out->es)
        return fail(ctx, SKEL_ERR_TYPE, "output element size != sizeof(result)");
    TRY(check_args(ctx, m, args, nargs));
    TRY(ensure_device(a));
    TRY(ensure_device(b));
    TRY(wait_dl(b));  // both are rewritten
    TRY(wait_dl(out));
    const size_t n = a->n, esa = a->es, esb = b->es, eso = out->es;
    if (out != a) {
        if (out->n != n) {
            out->n = n;
            if (out->host) {
                cudaFreeHost(out->host);
                out->host = nullptr;
            }
        }
        out->dist = SKEL_COPY;
        TRY(place(out, SKEL_COPY));
    }
    const int block = (int)m->sig[9];
    const uint64_t E = m->sig[8];
    std::vector<unsigned char> abuf;
    struct Ptrs {
        void *p[16];
    };
    auto launch = [&](Slot &s, size_t li, const Ptrs &bs, void *bown, const Ptrs &os, const void *pa,
                      uint64_t cnt) -> int {
        int vec_ok = al16(pa) && al16(bown);
        for (int j = 0; j < D; ++j) vec_ok = vec_ok && al16(bs.p[j]) && al16(os.p[j]);
        pack_args(m, args, nargs, li, abuf);
        const size_t chunks = vec_ok ? std::max<uint64_t>(cnt / E, 1) : cnt;
        const int grid = ew_grid(s, chunks, block);
        int nsrc = D, ndst = D, op = (int)combine;
        void *params[] = {&pa, (void *)&bs, &nsrc, &bown, (void *)&os, &ndst, &cnt, &op, &vec_ok, abuf.data()};
        DevGuard g(s.dev);
        CK(ctx, launch_dependent((const void *)m->k_zipcomb, dim3(grid), dim3(block), params, s.stream));
        ctx->stats.kernel_launches++;
        ctx->stats.d2d_bytes += (uint64_t)(D - 1) * cnt * (esb + eso);
        return SKEL_OK;
    };
    // NVSwitch multicast form (skel_zipcomb_mm_kernel): float32 '+' combine and
    // 4-byte elements, every local slot on its own multicast-capable device,
    // b's and out's buffers VMM allocations bound to one multicast object each
    bool mm = !ctx->rank_mode && m->k_zipcomb_mm && b->dt == SKEL_DT_F32 && combine == SKEL_COMBINE_ADD &&
              esa == 4 && eso == 4 && E == 4;
    if (mm) {
        TRY(join(ctx));
        mm = mc_bind(b, full_bytes(b)) && mc_bind(out, full_bytes(out));
    }
    if (mm) {
        for (size_t li = 0; li < ctx->slots.size(); ++li) {
            Slot &s = ctx->slots[li];
            const int k = s.d;
            uint64_t cnt = want_count(a, SKEL_BLOCK, k);
            const size_t lo = part_lo(a, k);
            if (!cnt) continue;
            const void *pa = a->dist == SKEL_COPY ? a->bufs[li].base + lo * esa : a->bufs[li].ptr(esa);
            const float *mcb = reinterpret_cast<const float *>(b->mc.va) + lo;
            void *bown = b->bufs[li].base + lo * esb;
            float *mco = reinterpret_cast<float *>(out->mc.va) + lo;
            int vec_ok = al16(pa) && al16(mcb) && al16(bown) && al16(mco);
            pack_args(m, args, nargs, li, abuf);
            const uint64_t work = vec_ok ? cnt / 4 : cnt;
            const int grid = ew_grid(s, std::max<uint64_t>(work, 1), block);
            uint64_t ncall = cnt;
            void *params[] = {&pa, &mcb, &bown, &mco, &ncall, &vec_ok, abuf.data()};
            DevGuard g(s.dev);
            CK(ctx, launch_dependent((const void *)m->k_zipcomb_mm, dim3(grid), dim3(block), params, s.stream));
            ctx->stats.kernel_launches++;
            ctx->stats.multimem_launches++;
            ctx->stats.d2d_bytes += (uint64_t)cnt * (esb + eso);
        }
        TRY(join(ctx));
    } else if (!ctx->rank_mode) {
        TRY(join(ctx));
        for (size_t li = 0; li < ctx->slots.size(); ++li) {
            Slot &s = ctx->slots[li];
            const int k = s.d;
            const size_t lo = part_lo(a, k), cnt = want_count(a, SKEL_BLOCK, k);
            if (!cnt) continue;
            Ptrs bs{}, os{};
            for (int j = 0; j < D; ++j) {
                bs.p[j] = b->bufs[j].base + lo * esb;
                os.p[j] = out->bufs[j].base + lo * eso;
            }
            const void *pa = a->dist == SKEL_COPY ? a->bufs[li].base + lo * esa : a->bufs[li].ptr(esa);
            TRY(launch(s, li, bs, b->bufs[li].base + lo * esb, os, pa, cnt));
        }
        TRY(join(ctx));
    } else {
        Slot &s = ctx->slots[0];
        const int k = ctx->rank;
        // peers: NCCL symmetric windows (SKEL_NCCL_WINDOWS=1), else CUDA IPC
        bool win = false;
        if (ctx->nccl_windows) {
            bool wb = false, wo = false;
            TRY(win_setup(ctx, s, b, &wb));
            if (wb) TRY(win_setup(ctx, s, out, &wo));
            win = wb && wo;
        }
        const WinRec *wrb = win ? &ctx->wins[b->bufs[0].base] : nullptr;
        const WinRec *wro = win ? &ctx->wins[out->bufs[0].base] : nullptr;
        if (!win) {
            // a buffer that moved into ncclMemAlloc memory for a window NCCL then
            // declined has no CUDA IPC handle: the unfused sequence (every rank
            // decides alike -- the window outcomes were agreed)
            if (ctx->nccl_mem.count(b->bufs[0].base) || ctx->nccl_mem.count(out->bufs[0].base)) return unfused();
            TRY(ipc_peers(ctx, s, b->bufs[0]));
            TRY(ipc_peers(ctx, s, out->bufs[0]));
        }
        TRY(rank_barrier(ctx, s));  // every rank's copy of b is complete
        const size_t lo = part_lo(a, k), cnt = want_count(a, SKEL_BLOCK, k);
        const void *pa = a->dist == SKEL_COPY ? a->bufs[0].base + lo * esa : a->bufs[0].ptr(esa);
        const bool mm_rank = win && wrb->mc && wro->mc && m->k_zipcomb_mm && b->dt == SKEL_DT_F32 &&
                             combine == SKEL_COMBINE_ADD && esa == 4 && eso == 4 && E == 4;
        if (cnt && mm_rank) {  // NVLS through the windows' multicast addresses
            const float *mcb = reinterpret_cast<const float *>(wrb->mc) + lo;
            float *mco = reinterpret_cast<float *>(wro->mc) + lo;
            void *bown = b->bufs[0].base + lo * esb;
            int vec_ok = al16(pa) && al16(mcb) && al16(bown) && al16(mco);
            pack_args(m, args, nargs, 0, abuf);
            const int grid = ew_grid(s, std::max<uint64_t>(vec_ok ? cnt / 4 : cnt, 1), block);
            uint64_t ncall = cnt;
            void *params[] = {&pa, &mcb, &bown, &mco, &ncall, &vec_ok, abuf.data()};
            DevGuard g(s.dev);
            CK(ctx, launch_dependent((const void *)m->k_zipcomb_mm, dim3(grid), dim3(block), params, s.stream));
            ctx->stats.kernel_launches++;
            ctx->stats.multimem_launches++;
        } else if (cnt) {
            Ptrs bs{}, os{};
            for (int j = 0; j < D; ++j) {
                bs.p[j] = (win ? wrb->peers[j] : b->bufs[0].peers[j]) + lo * esb;
                os.p[j] = (win ? wro->peers[j] : out->bufs[0].peers[j]) + lo * eso;
            }
            TRY(launch(s, 0, bs, b->bufs[0].base + lo * esb, os, pa, cnt));
        }
        TRY(rank_barrier(ctx, s));  // every rank's part of out has landed everywhere
    }
    for (size_t li = 0; li < ctx->slots.size(); ++li) {
        const int k = ctx->slots[li].d;
        b->bufs[li].off = part_lo(b, k);
        b->bufs[li].count = want_count(b, SKEL_BLOCK, k);
        out->bufs[li].off = 0;
        out->bufs[li].count = n;
    }
    b->dist = SKEL_BLOCK;
    b->dev_valid = true;
    b->diverged = false;
    device_wrote(b);
    out->dist = SKEL_COPY;
    out->dev_valid = true;
    out->diverged = false;
    device_wrote(out);
    return SKEL_OK;
}

int skel_reduce_to(skel_ctx_t ctx, const char *src, skel_vec_t in, skel_vec_t result, const skel_arg *args,
                   int nargs) {
    SKEL_RANGE("skel_reduce_to");
    if (!ctx || !src || !in || !result || in->ctx != ctx || result->ctx != ctx || (nargs && !args) || nargs < 0)
        return fail(ctx, SKEL_ERR_ARG, "bad reduce arguments");
    if (in->n == 0) return fail(ctx, SKEL_ERR_SIZE, "reduce of an empty vector (eq. 3 has no identity)");
    Module *m = nullptr;
    TRY(get_module(ctx, Kind::Red, src, &m));
    TRY(check_red(ctx, m, in));
    if (result->es != in->es) return fail(ctx, SKEL_ERR_TYPE, "result element size != input element size");
    TRY(check_args(ctx, m, args, nargs));
    TRY(ensure_device(in));
    // the result is a 1-element vector with a copy on every local device
    if (result->n != 1) {
        result->n = 1;
        if (result->host) {
            cudaFreeHost(result->host);
            result->host = nullptr;
        }
    }
    TRY(wait_dl(result));
    result->dist = SKEL_COPY;
    TRY(place(result, SKEL_COPY));
    std::vector<RedLayout> Ls;
    if (ctx->D == 1) {
        // one device: the Reduce kernel writes the result element itself
        TRY(reduce_core(ctx, m, in, args, nargs, Ls, result->bufs[0].ptr(result->es)));
    } else {
        TRY(reduce_core(ctx, m, in, args, nargs, Ls));
        TRY(finish_scalar(ctx, in, Ls));
        for (size_t li = 0; li < ctx->slots.size(); ++li) {
            Slot &s = ctx->slots[li];
            DevGuard g(s.dev);
            CK(ctx, cudaMemcpyAsync(result->bufs[li].ptr(result->es), s.ws + Ls[li].o_fold, in->es,
                                    cudaMemcpyDeviceToDevice, s.stream));
        }
    }
    result->dev_valid = true;
    device_wrote(result);
    result->diverged = false;
    return SKEL_OK;
}

int skel_reduce(skel_ctx_t ctx, const char *src, skel_vec_t in, void *result_host, const skel_arg *args, int nargs) {
    SKEL_RANGE("skel_reduce");
    if (!ctx || !src || !in || !result_host || in->ctx != ctx || (nargs && !args) || nargs < 0)
        return fail(ctx, SKEL_ERR_ARG, "bad reduce arguments");
    if (in->n == 0) return fail(ctx, SKEL_ERR_SIZE, "reduce of an empty vector (eq. 3 has no identity)");
    Module *m = nullptr;
    TRY(get_module(ctx, Kind::Red, src, &m));
    TRY(check_red(ctx, m, in));
    TRY(check_args(ctx, m, args, nargs));
    TRY(ensure_device(in));
    std::vector<RedLayout> Ls;
    TRY(reduce_core(ctx, m, in, args, nargs, Ls));
    TRY(finish_scalar(ctx, in, Ls));
    // Scalar::getValue
    Slot &s = ctx->slots[0];
    DevGuard g(s.dev);
    CK(ctx, cudaMemcpyAsync(result_host, s.ws + Ls[0].o_fold, in->es, cudaMemcpyDeviceToHost, s.stream));
    ctx->stats.d2h_bytes += in->es;
    ctx->stats.d2h_copies++;
    return sync_all(ctx);
}

int skel_scan(skel_ctx_t ctx, const char *src, skel_vec_t in, skel_vec_t out, const void *identity,
              const skel_arg *args, int nargs) {
    SKEL_RANGE("skel_scan");
    if (!ctx || !src || !in || !out || !identity || in->ctx != ctx || out->ctx != ctx || (nargs && !args) ||
        nargs < 0)
        return fail(ctx, SKEL_ERR_ARG, "bad scan arguments");
    Module *m = nullptr;
    TRY(get_module(ctx, Kind::Red, src, &m));
    TRY(check_red(ctx, m, in));
    if (out->es != in->es) return fail(ctx, SKEL_ERR_TYPE, "output element size != input element size");
    TRY(check_args(ctx, m, args, nargs));
    TRY(ensure_device(in));
    TRY(prepare_output(out, in->n, in->dist, out == in));
    if (in->n == 0) return SKEL_OK;
    const int D = ctx->D;
    const bool cross = D > 1 && in->dist == SKEL_BLOCK;
    std::vector<RedLayout> Ls(ctx->slots.size());
    std::vector<unsigned char> abuf;
    // seeds: device k starts from agg_0 (+) ... (+) agg_{k-1} (one exchange of
    // D partial results)
    const uint64_t SRB = m->sig[15] & 0xffff;  // rows (consumer threads) per scan tile
    const uint64_t TILE = SRB * m->sig[8];      // scan tile (elements)
    const uint64_t CH = (m->sig[15] >> 16) & 0xffff;                     // tiles per CTA per slice
    const uint64_t REPL = std::max<uint64_t>(1, (m->sig[15] >> 32) & 0xff);  // copies of each status word
    const bool packed = m->sig[13] != 0;
    TRY(set_smem_attr(ctx, m, ctx->slots[0]));
    int occ = 1;  // persistent grid: SMs x resident CTAs per SM
    {
        DevGuard g(ctx->slots[0].dev);
        if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, (const void *)m->k_scan, (int)m->sig[14],
                                                          (size_t)m->sig[12]) != cudaSuccess || occ < 1) {
            cudaGetLastError();
            occ = 1;
        }
    }
    // A window folds G-1 aggregates with one warp, at most 32 x AGG_PER = 512 of
    // them (red.cuh), so the grid is capped at 513 CTAs (the kernel traps above)
    constexpr uint64_t kScanMaxGrid = 32 * 16 + 1;
    auto scan_grid = [&](const Slot &s) -> uint64_t {
        return std::min<uint64_t>((uint64_t)s.sms * (uint64_t)occ, kScanMaxGrid);
    };
    // one aggregate status word per (slice, CTA)
    auto scan_slots = [&](const Slot &s, uint64_t cnt) -> uint64_t {
        const uint64_t per_slice = scan_grid(s) * CH, nft = cnt / TILE;
        return std::max<uint64_t>(1, (nft + per_slice - 1) / per_slice) * scan_grid(s);
    };
    // small vectors: two short launches (tile aggregates, seeded tile scans)
    // instead of the persistent pipeline; SKEL_SCAN_SMALL_MAX
    // (elements, a tuning hook) moves the switch point.  Default: up to 8 MiB of
    // elements (2^21 floats); from 2^22 floats the persistent Scan is faster
    // (14.4 vs 15.2 us, profiles/r01_scan_crossover_s4.txt)
    static const uint64_t small_max_env = [] {
        const char *e = getenv("SKEL_SCAN_SMALL_MAX");
        return e ? (uint64_t)strtoull(e, nullptr, 10) : ~0ull;
    }();
    const uint64_t SM_TILE = m->sig[9] * ((m->sig[15] >> 50) & 0xff);  // reduce block x elements per thread
    const uint64_t small_max = small_max_env != ~0ull ? small_max_env : (uint64_t)(2u << 20) * 4 / m->sig[3];
    auto small_scan = [&](uint64_t cnt) { return m->k_scan_small && SM_TILE > 0 && cnt <= small_max; };
    for (size_t li = 0; li < ctx->slots.size(); ++li) {
        Slot &s = ctx->slots[li];
        const uint64_t cnt = in->bufs[li].count;
        Ls[li] = red_layout(m, D, red_parts(m, s, cnt), scan_slots(s, cnt));
        // room for the small path's tile aggregates also when the persistent
        // kernel is chosen: it falls back to the small path if the cooperative
        // launch cannot make its grid co-resident
        const size_t extra = SM_TILE > 0 ? (size_t)((cnt + SM_TILE - 1) / SM_TILE) * Ls[li].slot : 0;
        TRY(ensure_ws(ctx, s, Ls[li].total + extra));
    }
    if (cross) {
        std::vector<RedLayout> Lr;
        TRY(reduce_core(ctx, m, in, args, nargs, Lr));
    }

    std::vector<unsigned char> idbuf(align_up(m->sig[4], 16), 0);
    memcpy(idbuf.data(), identity, in->es);
    for (size_t li = 0; li < ctx->slots.size(); ++li) {
        Slot &s = ctx->slots[li];
        uint64_t cnt = in->bufs[li].count;
        if (!cnt) continue;
        const size_t G = (size_t)scan_grid(s);
        const RedLayout &L = Ls[li];
        TRY(ensure_status(ctx, s, REPL * (scan_slots(s, cnt) + 64), packed));
        TRY(set_smem_attr(ctx, m, s));
        pack_args(m, args, nargs, li, abuf);
        DevGuard g(s.dev);
        const void *seed = nullptr;
        if (cross) {
            const void *aggs = s.ws + L.o_gather;
            int k = s.d;
            void *seedp = s.ws + L.o_seed;
            void *params[] = {&aggs, &k, idbuf.data(), &seedp, abuf.data()};
            CK(ctx, launch_dependent((const void *)m->k_seed, dim3(1), dim3(32), params, s.stream));
            ctx->stats.kernel_launches++;
            seed = seedp;
        }
        const void *pin = in->bufs[li].ptr(in->es);
        void *pout = out->bufs[li].ptr(out->es);
        bool small = small_scan(cnt);
        if (!small) {
            // The persistent Scan's windows wait on aggregates of higher-index
            // CTAs, so the whole grid must be resident at once: launch it
            // cooperatively (the driver guarantees co-residency or refuses).
            // Persistent Scans of logical devices that share one GPU run one
            // after another (event chain) so their grids never interleave.
            for (size_t lj = 0; lj < li; ++lj)
                if (ctx->slots[lj].dev == s.dev && ctx->slots[lj].ev_scan_live)
                    CK(ctx, cudaStreamWaitEvent(s.stream, ctx->slots[lj].ev_scan, 0));
            CUtensorMap tin, tout;
            const uint64_t rows = (cnt / TILE) * SRB;
            int use_tma = m->sig[5] && make_tmap(&tin, pin, rows, (uint32_t)(SRB / 2)) &&
                          make_tmap(&tout, pout, rows, (uint32_t)(SRB / 2));
            void *status = s.st64, *flags = s.fl32, *aggv = s.ws + L.o_aggv, *incv = s.ws + L.o_incv;
            unsigned *counters = s.counters;
            unsigned *epoch_ptr = s.counters + 3;  // device-resident scan epoch (graph-replay safe)
            void *total = nullptr;
            void *params[] = {&tin, &tout, &pin, &pout, &cnt, &use_tma, idbuf.data(), &seed, &status, &flags,
                              &aggv, &incv, &counters, &epoch_ptr, &total, abuf.data()};
            cudaLaunchConfig_t cfg = {};
            cfg.gridDim = dim3((unsigned)G);
            cfg.blockDim = dim3((unsigned)m->sig[14]);
            cfg.dynamicSmemBytes = use_tma ? m->sig[12] : 0;
            cfg.stream = s.stream;
            cudaLaunchAttribute attr[2];
            attr[0].id = cudaLaunchAttributeCooperative;
            attr[0].val.cooperative = 1;
            attr[1].id = cudaLaunchAttributeProgrammaticStreamSerialization;
            attr[1].val.programmaticStreamSerializationAllowed = 1;
            cfg.attrs = attr;
            cfg.numAttrs = pdl_enabled() ? 2 : 1;
            cudaError_t le = cudaLaunchKernelExC(&cfg, (const void *)m->k_scan, params);
            if (le != cudaSuccess && le != cudaErrorCooperativeLaunchTooLarge && cfg.numAttrs == 2) {
                cudaGetLastError();  // the driver declined the pair of attributes: cooperative only
                cfg.numAttrs = 1;
                le = cudaLaunchKernelExC(&cfg, (const void *)m->k_scan, params);
            }
            if (le == cudaErrorCooperativeLaunchTooLarge) {
                cudaGetLastError();  // fewer SMs than queried (MPS / green context): two short launches
                ctx->stats.scan_coop_fallbacks++;
                small = true;
            } else {
                CK(ctx, le);
                CK(ctx, cudaEventRecord(s.ev_scan, s.stream));
                s.ev_scan_live = true;
                ctx->stats.kernel_launches++;
            }
        }
        if (small && SM_TILE > 0) {
            const unsigned nt = (unsigned)((cnt + SM_TILE - 1) / SM_TILE);
            void *aggs = s.ws + L.total;
            int early = 0;
            void *pa[] = {&pin, &cnt, &aggs, &early, abuf.data()};
            CK(ctx, cudaLaunchKernel((const void *)m->k_scan_agg, dim3(nt), dim3((unsigned)m->sig[9]), pa, 0, s.stream));
            const void *caggs = aggs;
            void *ps[] = {&pin, &pout, &cnt, &caggs, idbuf.data(), &seed, abuf.data()};
            CK(ctx, launch_dependent((const void *)m->k_scan_small, dim3(nt), dim3((unsigned)m->sig[9]), ps, s.stream));
            ctx->stats.kernel_launches += 2;
        } else if (small) {
            return fail(ctx, SKEL_ERR_CUDA, "persistent Scan grid cannot be co-resident and this module has no "
                                            "small-vector path");
        }
    }
    out->dev_valid = true;
    device_wrote(out);
    return SKEL_OK;
}

int skel_prepare(skel_ctx_t ctx, const char *kind, const char *src) {
    if (!ctx || !kind || !src) return fail(ctx, SKEL_ERR_ARG, "bad arguments");
    Kind k;
    if (!strcmp(kind, "map")) k = Kind::Map;
    else if (!strcmp(kind, "zip")) k = Kind::Zip;
    else if (!strcmp(kind, "reduce") || !strcmp(kind, "scan")) k = Kind::Red;
    else if (!strcmp(kind, "index")) k = Kind::Idx;
    else if (!strcmp(kind, "lanes")) k = Kind::Lanes;
    else return fail(ctx, SKEL_ERR_ARG, "kind must be map|zip|reduce|scan|index|lanes");
    Module *m = nullptr;
    return get_module(ctx, k, src, &m);
}

// ---- CUDA graphs: capture a skeleton sequence once, replay it ------------------------
int skel_capture_begin(skel_ctx_t ctx) {
    if (!ctx) return fail(nullptr, SKEL_ERR_ARG, "ctx is NULL");
    if (ctx->capturing) return fail(ctx, SKEL_ERR_STATE, "already capturing");
    TRY(sync_all(ctx));
    Slot &s0 = ctx->slots[0];
    {
        DevGuard g(s0.dev);
        CK(ctx, cudaStreamBeginCapture(s0.stream, cudaStreamCaptureModeRelaxed));
        CK(ctx, cudaEventRecord(s0.ev, s0.stream));
    }
    for (size_t li = 1; li < ctx->slots.size(); ++li) {  // fork: the other streams join the capture
        DevGuard g(ctx->slots[li].dev);
        CK(ctx, cudaStreamWaitEvent(ctx->slots[li].stream, s0.ev, 0));
    }
    ctx->captured.clear();
    ctx->capturing = true;
    return SKEL_OK;
}

int skel_capture_end(skel_ctx_t ctx, skel_graph_t *out) {
    if (!ctx || !out) return fail(ctx, SKEL_ERR_ARG, "bad arguments");
    if (!ctx->capturing) return fail(ctx, SKEL_ERR_STATE, "not capturing");
    ctx->capturing = false;
    Slot &s0 = ctx->slots[0];
    for (size_t li = 1; li < ctx->slots.size(); ++li) {  // join back into the origin stream
        Slot &s = ctx->slots[li];
        DevGuard g(s.dev);
        CK(ctx, cudaEventRecord(s.ev, s.stream));
        DevGuard g0(s0.dev);
        CK(ctx, cudaStreamWaitEvent(s0.stream, s.ev, 0));
    }
    DevGuard g(s0.dev);
    auto *gr = new skel_graph_s();
    gr->ctx = ctx;
    cudaError_t e = cudaStreamEndCapture(s0.stream, &gr->graph);
    if (e == cudaSuccess) e = cudaGraphInstantiate(&gr->exec, gr->graph, 0);
    if (e != cudaSuccess) {
        if (gr->graph) cudaGraphDestroy(gr->graph);
        delete gr;
        return fail(ctx, SKEL_ERR_CUDA, std::string("capture: ") + cudaGetErrorString(e));
    }
    gr->written.swap(ctx->captured);
    *out = gr;
    return SKEL_OK;
}

int skel_graph_launch(skel_graph_t g) {
    SKEL_RANGE("skel_graph_launch");
    if (!g) return fail(nullptr, SKEL_ERR_ARG, "graph is NULL");
    skel_ctx_s *ctx = g->ctx;
    Slot &s0 = ctx->slots[0];
    for (size_t li = 1; li < ctx->slots.size(); ++li) {  // earlier work on the other streams first
        Slot &s = ctx->slots[li];
        DevGuard gd(s.dev);
        CK(ctx, cudaEventRecord(s.ev, s.stream));
        DevGuard g0(s0.dev);
        CK(ctx, cudaStreamWaitEvent(s0.stream, s.ev, 0));
    }
    {
        DevGuard gd(s0.dev);
        CK(ctx, cudaGraphLaunch(g->exec, s0.stream));
        CK(ctx, cudaEventRecord(s0.ev, s0.stream));
    }
    for (size_t li = 1; li < ctx->slots.size(); ++li) {  // later work on the other streams after it
        DevGuard gd(ctx->slots[li].dev);
        CK(ctx, cudaStreamWaitEvent(ctx->slots[li].stream, s0.ev, 0));
    }
    for (auto &w : g->written)  // the replay rewrote these vectors on the devices
        if (ctx->vecs.count(w.first) && w.first->serial == w.second) {
            w.first->host_valid = false;
            w.first->dev_valid = true;
        }
    return SKEL_OK;
}

int skel_graph_destroy(skel_graph_t g) {
    if (!g) return fail(nullptr, SKEL_ERR_ARG, "graph is NULL");
    if (g->exec) cudaGraphExecDestroy(g->exec);
    if (g->graph) cudaGraphDestroy(g->graph);
    delete g;
    return SKEL_OK;
}

// ---- pure host logic -------------------------------------------------------------
int skel_entry_name(const char *src, char *name, size_t cap) {
    if (!src || !name || cap == 0) return fail(nullptr, SKEL_ERR_ARG, "bad arguments");
    std::string err;
    std::string e = entry_name(src, &err);
    if (e.empty()) return fail(nullptr, SKEL_ERR_COMPILE, err);
    if (e.size() + 1 > cap) return fail(nullptr, SKEL_ERR_SIZE, "name buffer too small");
    memcpy(name, e.c_str(), e.size() + 1);
    return SKEL_OK;
}

int skel_compile_check(const char *kind, const char *src, int fmad, char *log, size_t cap, size_t *cubin_bytes) {
    if (!kind || !src) return fail(nullptr, SKEL_ERR_ARG, "bad arguments");
    Kind k;
    if (!strcmp(kind, "map")) k = Kind::Map;
    else if (!strcmp(kind, "zip")) k = Kind::Zip;
    else if (!strcmp(kind, "reduce") || !strcmp(kind, "scan")) k = Kind::Red;
    else if (!strcmp(kind, "index")) k = Kind::Idx;
    else if (!strcmp(kind, "lanes")) k = Kind::Lanes;
    else return fail(nullptr, SKEL_ERR_ARG, "kind must be map|zip|reduce|scan|index|lanes");
    std::string l;
    std::vector<char> cubin;
    const int st = compile_only(k, src, 256, fmad != 0, &l, &cubin);
    if (log && cap) {
        const size_t m = std::min(cap - 1, l.size());
        memcpy(log, l.data(), m);
        log[m] = 0;
    }
    if (cubin_bytes) *cubin_bytes = cubin.size();
    if (st != SKEL_OK) g_last_error = l;
    const char *dump = getenv("SKEL_DUMP_CUBIN");  // inspection: cuobjdump -sass / -res-usage
    if (st == SKEL_OK && dump && *dump) {
        FILE *f = fopen(dump, "wb");
        if (f) {
            fwrite(cubin.data(), 1, cubin.size(), f);
            fclose(f);
        }
    }
    return st;
}

int skel_plan_part(size_t n, int D, int k, size_t *lo, size_t *hi) {
    if (D < 1 || k < 0 || k >= D || !lo || !hi) return fail(nullptr, SKEL_ERR_ARG, "bad arguments");
    part_range(n, D, k, lo, hi);
    return SKEL_OK;
}

int skel_plan_exchange(skel_dist from, skel_dist to, skel_combine combine, int *xchg) {
    if (!xchg || (int)from < 0 || (int)from > 2 || (int)to < 0 || (int)to > 2 || (int)combine < 0 || (int)combine > 4)
        return fail(nullptr, SKEL_ERR_ARG, "bad arguments");
    const int x = plan_exchange(from, to, combine);
    if (x < 0) return fail(nullptr, SKEL_ERR_STATE, "combine requires a copy-distributed source");
    *xchg = x;
    return SKEL_OK;
}

}  // extern "C"
