// jit.cpp -- NVRTC injection of user functions into the skeleton templates,
// plus the in-memory and on-disk kernel caches.
//
// PAPER.md: "User-defined customizing functions passed to the skeletons are
// merged with pre-implemented skeleton code during code generation"
// (P:L174-181); "SkelCL saves already compiled kernels on disk. They can be
// loaded later if the same kernel is used again".
//
// Here the generated translation unit is
//     prelude.cuh + user source + "#define SKEL_FN <entry>" + map.cuh|red.cuh
// compiled by NVRTC straight to an sm_100a cubin (no PTX JIT at load time),
// loaded with cudaLibraryLoadData (context-independent: one load serves every
// device of the process), and its signature table `skel_sig` is read back
// once to validate element sizes and to lay out the Arguments buffer.
#include <nvrtc.h>
#include <sys/stat.h>
#include <unistd.h>

#include <chrono>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <fstream>
#include <sstream>

#include "internal.h"
#include "templates.inc"  // generated at build time: kPreludeSrc, kMapSrc, kRedSrc

namespace skelrt {

static uint64_t fnv1a(const std::string &s, uint64_t h) {
    for (unsigned char c : s) {
        h ^= c;
        h *= 1099511628211ull;
    }
    return h;
}

static std::string hexkey(const std::string &s) {
    char buf[40];
    snprintf(buf, sizeof buf, "%016llx%016llx", (unsigned long long)fnv1a(s, 1469598103934665603ull),
             (unsigned long long)fnv1a(s, 0x9e3779b97f4a7c15ull));
    return buf;
}

// Last top-level function definition of a C/C++ source: the identifier in
// front of the parameter list of the last `(...) {` at brace depth 0.
// Comments, string/char literals and preprocessor lines are skipped.
std::string entry_name(const std::string &src, std::string *err) {
    std::string clean;
    clean.reserve(src.size());
    const size_t n = src.size();
    bool line_start = true;
    for (size_t i = 0; i < n;) {
        char c = src[i];
        if (line_start) {
            size_t j = i;
            while (j < n && (src[j] == ' ' || src[j] == '\t')) ++j;
            if (j < n && src[j] == '#') {  // preprocessor line (with continuations)
                while (j < n && src[j] != '\n') {
                    if (src[j] == '\\' && j + 1 < n && src[j + 1] == '\n') ++j;
                    ++j;
                }
                i = j;
                clean.push_back(' ');
                continue;
            }
        }
        if (c == '/' && i + 1 < n && src[i + 1] == '/') {
            while (i < n && src[i] != '\n') ++i;
            continue;
        }
        if (c == '/' && i + 1 < n && src[i + 1] == '*') {
            i += 2;
            while (i + 1 < n && !(src[i] == '*' && src[i + 1] == '/')) ++i;
            i += 2;
            clean.push_back(' ');
            continue;
        }
        if (c == '"' || c == '\'') {
            const char q = c;
            ++i;
            while (i < n && src[i] != q) {
                if (src[i] == '\\') ++i;
                ++i;
            }
            ++i;
            clean.push_back(' ');
            continue;
        }
        line_start = (c == '\n');
        clean.push_back(c);
        ++i;
    }
    int depth = 0;
    std::string last;
    for (size_t i = 0; i < clean.size(); ++i) {
        const char c = clean[i];
        if (c == '{') {
            if (depth == 0) {
                // walk back over whitespace and trailing qualifiers to ')'
                long j = (long)i - 1;
                for (;;) {
                    while (j >= 0 && isspace((unsigned char)clean[j])) --j;
                    long e = j;
                    while (j >= 0 && (isalnum((unsigned char)clean[j]) || clean[j] == '_')) --j;
                    std::string word = clean.substr(j + 1, e - j);
                    if (word == "const" || word == "noexcept" || word == "__restrict__") continue;
                    j = e;
                    break;
                }
                if (j >= 0 && clean[j] == ')') {
                    int pd = 0;
                    long k = j;
                    for (; k >= 0; --k) {
                        if (clean[k] == ')') ++pd;
                        else if (clean[k] == '(') {
                            if (--pd == 0) break;
                        }
                    }
                    long e = k - 1;
                    while (e >= 0 && isspace((unsigned char)clean[e])) --e;
                    long b = e;
                    while (b >= 0 && (isalnum((unsigned char)clean[b]) || clean[b] == '_')) --b;
                    std::string name = clean.substr(b + 1, e - b);
                    if (!name.empty() && name != "if" && name != "for" && name != "while" && name != "switch" &&
                        !isdigit((unsigned char)name[0]))
                        last = name;
                }
            }
            ++depth;
        } else if (c == '}') {
            --depth;
        }
    }
    if (last.empty() && err) *err = "no top-level function definition found in the user function source";
    return last;
}

int get_module_slow(skel_ctx_s *ctx, Kind kind, const char *src, Module **out);

static const char *kind_name(Kind k) {
    switch (k) {
        case Kind::Map: return "map";
        case Kind::Zip: return "zip";
        case Kind::Idx: return "idx";
        case Kind::Lanes: return "lanes";
        default: return "red";
    }
}

static std::string cache_dir(skel_ctx_s *ctx) {
    if (!ctx->disk_cache) return "";
    if (!ctx->cache_dir.empty()) return ctx->cache_dir;
    const char *e = getenv("SKEL_CACHE_DIR");
    if (e) return e;
    const char *home = getenv("HOME");
    return std::string(home ? home : "/tmp") + "/.cache/skel_b200";
}

static void mkdirs(const std::string &path) {
    std::string cur;
    std::stringstream ss(path);
    std::string part;
    if (!path.empty() && path[0] == '/') cur = "/";
    while (std::getline(ss, part, '/')) {
        if (part.empty()) continue;
        cur += part + "/";
        mkdir(cur.c_str(), 0755);
    }
}

static double ms_since(std::chrono::steady_clock::time_point t0) {
    return std::chrono::duration<double, std::milli>(std::chrono::steady_clock::now() - t0).count();
}

// prelude + user source + SKEL_FN + skeleton template
static int assemble(Kind kind, const std::string &user, int block, bool fmad, std::string *text,
                    std::vector<std::string> *opts, std::string *err) {
    const std::string entry = entry_name(user, err);
    if (entry.empty()) return SKEL_ERR_COMPILE;
    *opts = {"--gpu-architecture=sm_100a", "-default-device", "-std=c++17", "-lineinfo",
             fmad ? "--fmad=true" : "--fmad=false"};
    // tuning experiments: extra -D options for the skeleton templates (part of the cache key)
    if (const char *extra = getenv("SKEL_NVRTC_DEFINES")) {
        std::stringstream ss(extra);
        std::string tok;
        while (ss >> tok) opts->push_back(tok);
    }
    std::string defs;
    if (kind == Kind::Map) defs = "#define SKEL_NIN 1\n#define SKEL_BLOCK " + std::to_string(block) + "\n";
    if (kind == Kind::Zip) defs = "#define SKEL_NIN 2\n#define SKEL_BLOCK " + std::to_string(block) + "\n";
    if (kind == Kind::Idx) defs = "#define SKEL_NIN 0\n#define SKEL_BLOCK " + std::to_string(block) + "\n";
    if (kind == Kind::Lanes)
        defs = "#define SKEL_NIN 1\n#define SKEL_LANES 1\n#define SKEL_BLOCK " + std::to_string(block) + "\n";
    text->clear();
    text->reserve(user.size() + 65536);
    *text += "#line 1 \"skel_prelude.cuh\"\n";
    *text += kPreludeSrc;
    *text += "\n#line 1 \"user_function\"\n";
    *text += user;
    // "::entry": the user's function is a top-level one, so a template local of
    // the same name (e.g. a parameter `op`) cannot shadow it
    *text += "\n#line 1 \"skel_skeleton.cuh\"\n#define SKEL_FN ::" + entry + "\n" + defs;
    *text += (kind == Kind::Red) ? kRedSrc : kMapSrc;
    return SKEL_OK;
}

static int nvrtc_cubin(Kind kind, const std::string &text, const std::vector<std::string> &opts,
                       std::vector<char> *cubin, std::string *log) {
    nvrtcProgram prog;
    const std::string name = std::string("skel_") + kind_name(kind) + ".cu";
    if (nvrtcCreateProgram(&prog, text.c_str(), name.c_str(), 0, nullptr, nullptr) != NVRTC_SUCCESS) {
        *log = "nvrtcCreateProgram failed";
        return SKEL_ERR_COMPILE;
    }
    std::vector<const char *> copts;
    for (auto &o : opts) copts.push_back(o.c_str());
    nvrtcResult r = nvrtcCompileProgram(prog, (int)copts.size(), copts.data());
    size_t logsz = 0;
    nvrtcGetProgramLogSize(prog, &logsz);
    std::string l(logsz, '\0');
    if (logsz) nvrtcGetProgramLog(prog, &l[0]);
    if (r != NVRTC_SUCCESS) {
        *log = std::string("NVRTC: ") + nvrtcGetErrorString(r) + "\n" + l;
        nvrtcDestroyProgram(&prog);
        return SKEL_ERR_COMPILE;
    }
    size_t sz = 0;
    nvrtcGetCUBINSize(prog, &sz);
    cubin->resize(sz);
    nvrtcGetCUBIN(prog, cubin->data());
    nvrtcDestroyProgram(&prog);
    *log = l;
    return SKEL_OK;
}

int compile_only(Kind kind, const char *src, int block, bool fmad, std::string *log, std::vector<char> *cubin) {
    std::string text, err;
    std::vector<std::string> opts;
    if (assemble(kind, src, block, fmad, &text, &opts, &err) != SKEL_OK) {
        *log = err;
        return SKEL_ERR_COMPILE;
    }
    std::vector<char> tmp;
    return nvrtc_cubin(kind, text, opts, cubin ? cubin : &tmp, log);
}

int get_module(skel_ctx_s *ctx, Kind kind, const char *src, Module **out) {
    // fast path: the same user text with the same options was loaded before
    // (skips assembling and hashing the ~50 KB translation unit on every call)
    const char *extra = getenv("SKEL_NVRTC_DEFINES");
    std::string fast;
    fast.reserve(64 + strlen(src));
    fast += kind_name(kind);
    fast += '|';
    fast += std::to_string(ctx->block_size);
    fast += ctx->fmad ? "|f1|" : "|f0|";
    fast += extra ? extra : "";
    fast += '|';
    fast += src;
    auto fit = ctx->fast_modules.find(fast);
    if (fit != ctx->fast_modules.end()) {
        ctx->stats.compile_mem_hits++;
        *out = fit->second;
        return SKEL_OK;
    }
    if (ctx->capturing) {
        ctx->last_error = "user function not compiled yet: call skel_prepare (or run once) before capturing";
        return SKEL_ERR_STATE;
    }
    int st = get_module_slow(ctx, kind, src, out);
    if (st == SKEL_OK) ctx->fast_modules[fast] = *out;
    return st;
}

int get_module_slow(skel_ctx_s *ctx, Kind kind, const char *src, Module **out) {
    std::string err;
    const std::string user(src);
    const int block = ctx->block_size > 0 ? ctx->block_size : 256;
    std::string text;
    std::vector<std::string> opts;
    if (assemble(kind, user, block, ctx->fmad, &text, &opts, &err) != SKEL_OK) {
        ctx->last_error = err;
        return SKEL_ERR_COMPILE;
    }

    int maj = 0, min = 0;
    nvrtcVersion(&maj, &min);
    std::string keysrc = text;
    for (auto &o : opts) keysrc += "\n" + o;
    keysrc += "\nnvrtc " + std::to_string(maj) + "." + std::to_string(min);
    const std::string key = std::string(kind_name(kind)) + "_" + hexkey(keysrc);

    auto it = ctx->modules.find(key);
    if (it != ctx->modules.end()) {
        ctx->stats.compile_mem_hits++;
        *out = it->second.get();
        return SKEL_OK;
    }

    std::vector<char> cubin;
    const std::string dir = cache_dir(ctx);
    const std::string path = dir.empty() ? "" : dir + "/" + key + ".cubin";
    bool from_disk = false;
    auto t0 = std::chrono::steady_clock::now();
    if (!path.empty()) {
        std::ifstream f(path, std::ios::binary);
        if (f) {
            cubin.assign(std::istreambuf_iterator<char>(f), std::istreambuf_iterator<char>());
            from_disk = !cubin.empty();
        }
    }
    if (!from_disk) {
        std::string log;
        if (nvrtc_cubin(kind, text, opts, &cubin, &log) != SKEL_OK) {
            ctx->last_error = log;
            return SKEL_ERR_COMPILE;
        }
        ctx->stats.compile_misses++;
        ctx->stats.compile_ms += ms_since(t0);
        if (!path.empty()) {
            mkdirs(dir);
            const std::string tmp = path + ".tmp" + std::to_string(getpid());
            std::ofstream f(tmp, std::ios::binary);
            if (f) {
                f.write(cubin.data(), (std::streamsize)cubin.size());
                f.close();
                rename(tmp.c_str(), path.c_str());
            }
        }
    }

    auto m = std::make_unique<Module>();
    m->kind = kind;
    m->key = key;
    if (!path.empty() && !(getenv("SKEL_POLICY_CACHE") && atoi(getenv("SKEL_POLICY_CACHE")) == 0))
        m->policy_path = dir + "/" + key + ".policy";
    if (ctx->slots.empty()) {
        ctx->last_error = "context has no devices";
        return SKEL_ERR_STATE;
    }
    cudaSetDevice(ctx->slots[0].dev);
    cudaError_t ce = cudaLibraryLoadData(&m->lib, cubin.data(), nullptr, nullptr, 0, nullptr, nullptr, 0);
    if (ce != cudaSuccess) {
        ctx->last_error = std::string("cudaLibraryLoadData: ") + cudaGetErrorString(ce);
        return SKEL_ERR_CUDA;
    }
    auto getk = [&](const char *nm, cudaKernel_t *k) -> bool {
        cudaError_t e = cudaLibraryGetKernel(k, m->lib, nm);
        if (e != cudaSuccess) {
            ctx->last_error = std::string("cudaLibraryGetKernel(") + nm + "): " + cudaGetErrorString(e);
            return false;
        }
        return true;
    };
    if (kind == Kind::Red) {
        if (!getk("skel_reduce_kernel", &m->k_main) || !getk("skel_scan_kernel", &m->k_scan) ||
            !getk("skel_fold_kernel", &m->k_fold) || !getk("skel_seed_kernel", &m->k_seed) ||
            !getk("skel_scan_agg_kernel", &m->k_scan_agg) || !getk("skel_scan_small_kernel", &m->k_scan_small) ||
            !getk("skel_fold_aggs_kernel", &m->k_fold_aggs) || !getk("skel_red_agg2_kernel", &m->k_red_agg2))
            return SKEL_ERR_CUDA;
    } else {
        if (!getk("skel_ew_kernel", &m->k_main)) return SKEL_ERR_CUDA;
        if ((kind == Kind::Map || kind == Kind::Zip) && !getk("skel_ew_kernel_u1", &m->k_main_u1)) return SKEL_ERR_CUDA;
        if (kind == Kind::Zip && !getk("skel_zipcomb_kernel", &m->k_zipcomb)) return SKEL_ERR_CUDA;
        if (kind == Kind::Zip && !getk("skel_zipcomb_mm_kernel", &m->k_zipcomb_mm)) return SKEL_ERR_CUDA;
    }
    void *dsig = nullptr;
    size_t bytes = 0;
    ce = cudaLibraryGetGlobal(&dsig, &bytes, m->lib, "skel_sig");
    if (ce == cudaSuccess) ce = cudaMemcpy(m->sig, dsig, bytes < sizeof(m->sig) ? bytes : sizeof(m->sig),
                                           cudaMemcpyDeviceToHost);
    if (ce != cudaSuccess) {
        ctx->last_error = std::string("reading skel_sig: ") + cudaGetErrorString(ce);
        return SKEL_ERR_CUDA;
    }
    if (from_disk) {
        ctx->stats.compile_disk_hits++;
        ctx->stats.disk_load_ms += ms_since(t0);
    }
    *out = m.get();
    ctx->modules[key] = std::move(m);
    return SKEL_OK;
}

}  // namespace skelrt
