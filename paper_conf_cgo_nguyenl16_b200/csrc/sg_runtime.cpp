// sg_runtime.cpp -- NVRTC compilation, module management and the pipelined
// multi-GPU execution of a plan.
//
// Execution model (section 3.2.3, Fig. 3.5): the iteration
// range is cut into fragments; "partitions mapped to the same GPU run
// sequentially"; boundary streams of fragment n move to the consumer GPU while
// the producer GPU already computes fragment n+1.  Transfers are peer-to-peer
// -- over NVLink/NVSwitch on B200 -- on a dedicated copy
// stream per GPU, double-buffered (ring of `ring_depth` slots per cut edge),
// ordered by CUDA events only; the host never synchronises inside sg_run.
//
// Fragments never share state: every partition kernel recomputes the peek
// halo of its first tile (sg_codegen.cpp), and each cut-edge slot holds the
// whole window the consumer needs for the fragment (halo included).
#include "sg_runtime.h"

#include <dlfcn.h>
#include <nvrtc.h>
#include <sys/stat.h>

#include <algorithm>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <fstream>
#include <map>
#include <mutex>
#include <sstream>

namespace sg {

// ------------------------------------------------------- driver API shim
// libsg.so does not link libcuda: driver entry points are resolved through
// the runtime (cudaGetDriverEntryPoint) on first use, so the library loads on
// machines without a driver (CPU build/plan checks) and fails loudly at run.
namespace drv {
typedef CUresult (*PFN_load)(CUmodule*, const void*);
typedef CUresult (*PFN_getfn)(CUfunction*, CUmodule, const char*);
typedef CUresult (*PFN_setattr)(CUfunction, CUfunction_attribute, int);
typedef CUresult (*PFN_occ)(int*, CUfunction, int, size_t);
typedef CUresult (*PFN_launch)(CUfunction, unsigned, unsigned, unsigned, unsigned, unsigned, unsigned, unsigned,
                               CUstream, void**, void**);
typedef CUresult (*PFN_unload)(CUmodule);
typedef CUresult (*PFN_errstr)(CUresult, const char**);
typedef CUresult (*PFN_tmap)(CUtensorMap*, CUtensorMapDataType, cuuint32_t, void*, const cuuint64_t*, const cuuint64_t*,
                             const cuuint32_t*, const cuuint32_t*, CUtensorMapInterleave, CUtensorMapSwizzle,
                             CUtensorMapL2promotion, CUtensorMapFloatOOBfill);
struct Api {
    PFN_load load = nullptr;
    PFN_getfn getfn = nullptr;
    PFN_setattr setattr = nullptr;
    PFN_occ occ = nullptr;
    PFN_launch launch = nullptr;
    PFN_unload unload = nullptr;
    PFN_errstr errstr = nullptr;
    PFN_tmap tmap = nullptr;
};
static Api& api() {
    static Api a;
    static std::once_flag once;
    static std::string err;
    std::call_once(once, [] {
        auto get = [](const char* name, void** fp) {
            cudaDriverEntryPointQueryResult q;
            cudaError_t e = cudaGetDriverEntryPoint(name, fp, cudaEnableDefault, &q);
            if (e != cudaSuccess || q != cudaDriverEntryPointSuccess) { *fp = nullptr; cudaGetLastError(); }
        };
        get("cuModuleLoadData", (void**)&a.load);
        get("cuModuleGetFunction", (void**)&a.getfn);
        get("cuFuncSetAttribute", (void**)&a.setattr);
        get("cuOccupancyMaxActiveBlocksPerMultiprocessor", (void**)&a.occ);
        get("cuLaunchKernel", (void**)&a.launch);
        get("cuModuleUnload", (void**)&a.unload);
        get("cuGetErrorString", (void**)&a.errstr);
        get("cuTensorMapEncodeTiled", (void**)&a.tmap);
    });
    if (!a.load || !a.launch) throw Error(SG_E_CUDA, "CUDA driver not available (no GPU): the executor has no CPU fallback");
    return a;
}
}  // namespace drv

#define cuModuleLoadData drv::api().load
#define cuModuleGetFunction drv::api().getfn
#define cuFuncSetAttribute drv::api().setattr
#define cuOccupancyMaxActiveBlocksPerMultiprocessor drv::api().occ
#define cuLaunchKernel drv::api().launch
#define cuModuleUnload drv::api().unload
static const char* drv_errstr(CUresult r) {
    const char* s = nullptr;
    if (drv::api().errstr) drv::api().errstr(r, &s);
    return s ? s : "?";
}

#define SG_CU(x)                                                                          \
    do {                                                                                  \
        CUresult r_ = (x);                                                                \
        if (r_ != CUDA_SUCCESS) throw Error(SG_E_CUDA, std::string(#x) + ": " + drv_errstr(r_)); \
    } while (0)
#define SG_RT(x)                                                                          \
    do {                                                                                  \
        cudaError_t r_ = (x);                                                             \
        if (r_ != cudaSuccess) throw Error(SG_E_CUDA, std::string(#x) + ": " + cudaGetErrorString(r_)); \
    } while (0)

// ------------------------------------------------------------------ NVRTC
static std::mutex g_cache_mu;
static std::map<uint64_t, std::string> g_cubin_cache;

static uint64_t fnv1a(const std::string& s, uint64_t h = 1469598103934665603ULL) {
    for (unsigned char c : s) { h ^= c; h *= 1099511628211ULL; }
    return h;
}

std::string nvrtc_version() {
    int maj = 0, min = 0;
    nvrtcVersion(&maj, &min);
    return std::to_string(maj) + "." + std::to_string(min);
}

static std::string cache_dir() {
    const char* env = std::getenv("SG_CACHE_DIR");
    if (env && *env) return env;
    Dl_info info;
    if (dladdr((void*)&cache_dir, &info) && info.dli_fname) {
        std::string p = info.dli_fname;
        size_t k = p.rfind('/');
        if (k != std::string::npos) return p.substr(0, k) + "/.sg_cache";
    }
    return ".sg_cache";
}

static const char* kNvrtcOpts[] = {"--gpu-architecture=sm_100a", "--fmad=false",       "--std=c++17",
                                   "-default-device",            "--generate-line-info", "--prec-div=true",
                                   "--prec-sqrt=true",           "--ftz=false",         "-DSG_NVRTC=1"};

void compile_kernel(CompiledKernel& ck, int verbose) {
    std::string key_src = ck.ki.source + "\n//" + nvrtc_version();
    for (const char* o : kNvrtcOpts) key_src += o;
    key_src += kDeviceHeader;
    uint64_t key = fnv1a(key_src);
    {
        std::lock_guard<std::mutex> lk(g_cache_mu);
        auto it = g_cubin_cache.find(key);
        if (it != g_cubin_cache.end()) { ck.cubin = it->second; return; }
    }
    char hex[32];
    std::snprintf(hex, sizeof hex, "%016llx", (unsigned long long)key);
    std::string dir = cache_dir();
    std::string path = dir + "/" + hex + ".cubin";
    {
        std::ifstream in(path, std::ios::binary);
        if (in) {
            std::stringstream ss;
            ss << in.rdbuf();
            ck.cubin = ss.str();
            if (!ck.cubin.empty()) {
                std::lock_guard<std::mutex> lk(g_cache_mu);
                g_cubin_cache[key] = ck.cubin;
                return;
            }
        }
    }
    nvrtcProgram prog;
    const char* hdrs[] = {kDeviceHeader};
    const char* names[] = {"sg_device.cuh"};
    if (nvrtcCreateProgram(&prog, ck.ki.source.c_str(), (ck.ki.name + ".cu").c_str(), 1, hdrs, names) != NVRTC_SUCCESS)
        throw Error(SG_E_CUDA, "nvrtcCreateProgram failed");
    std::vector<const char*> opts(std::begin(kNvrtcOpts), std::end(kNvrtcOpts));
    if (verbose) opts.push_back("--ptxas-options=-v");
    nvrtcResult rc = nvrtcCompileProgram(prog, (int)opts.size(), opts.data());
    size_t logn = 0;
    nvrtcGetProgramLogSize(prog, &logn);
    std::string log(logn, '\0');
    if (logn) nvrtcGetProgramLog(prog, &log[0]);
    ck.log = log;
    if (rc != NVRTC_SUCCESS) {
        nvrtcDestroyProgram(&prog);
        if (verbose) std::fprintf(stderr, "%s\n", ck.ki.source.c_str());
        throw Error(SG_E_CUDA, "NVRTC failed for " + ck.ki.name + ":\n" + log.substr(0, 4000));
    }
    size_t n = 0;
    nvrtcGetCUBINSize(prog, &n);
    ck.cubin.assign(n, '\0');
    nvrtcGetCUBIN(prog, &ck.cubin[0]);
    nvrtcDestroyProgram(&prog);
    if (verbose && !log.empty()) std::fprintf(stderr, "[sg] %s: %s\n", ck.ki.name.c_str(), log.c_str());
    {
        std::lock_guard<std::mutex> lk(g_cache_mu);
        g_cubin_cache[key] = ck.cubin;
    }
    mkdir(dir.c_str(), 0755);
    std::string tmp = path + ".tmp" + std::to_string((unsigned long long)(uintptr_t)&ck);
    std::ofstream out(tmp, std::ios::binary);
    if (out) {
        out.write(ck.cubin.data(), (std::streamsize)ck.cubin.size());
        out.close();
        std::rename(tmp.c_str(), path.c_str());
    }
}

// ---------------------------------------------------------------- helpers
namespace {
struct DevGuard {
    int old = -1;
    explicit DevGuard(int dev) {
        if (cudaGetDevice(&old) != cudaSuccess) old = -1;
        SG_RT(cudaSetDevice(dev));
    }
    ~DevGuard() {
        if (old >= 0) cudaSetDevice(old);
    }
};

void ensure_module(CompiledKernel& ck, int dev) {
    if ((int)ck.fn.size() <= dev) {
        ck.mod.resize(dev + 1, nullptr);
        ck.fn.resize(dev + 1, nullptr);
        ck.fn_sync.resize(dev + 1, nullptr);
        ck.max_blocks_per_sm.resize(dev + 1, 0);
        ck.max_blocks_sync.resize(dev + 1, 0);
    }
    if (ck.fn[dev]) return;
    SG_RT(cudaFree(nullptr));  // make the primary context current
    SG_CU(cuModuleLoadData(&ck.mod[dev], ck.cubin.data()));
    auto setup = [&](const std::string& name, int threads, size_t smem, CUfunction& f, int& nb) {
        SG_CU(cuModuleGetFunction(&f, ck.mod[dev], name.c_str()));
        SG_CU(cuFuncSetAttribute(f, CU_FUNC_ATTRIBUTE_MAX_DYNAMIC_SHARED_SIZE_BYTES, (int)smem));
        SG_CU(cuOccupancyMaxActiveBlocksPerMultiprocessor(&nb, f, threads, smem));
        if (nb <= 0)
            throw Error(SG_E_SIZE, name + " cannot be resident (" + std::to_string(smem) + " B smem, " +
                                       std::to_string(threads) + " threads)");
    };
    setup(ck.ki.name, ck.ki.threads, ck.ki.smem, ck.fn[dev], ck.max_blocks_per_sm[dev]);
    if (ck.ki.mode == 1 && ck.ki.has_tma)
        setup(ck.ki.name_sync, ck.ki.threads_sync, ck.ki.smem_sync, ck.fn_sync[dev], ck.max_blocks_sync[dev]);
    if (ck.ki.mode == 2 && !ck.ki.name_start.empty())
        setup(ck.ki.name_start, ck.ki.threads, ck.ki.smem, ck.fn_sync[dev], ck.max_blocks_sync[dev]);
}

// 2-D row tensor map: dims {P items, rows}, box {P, box_rows}, 128B swizzle.
void encode_rows_map(CUtensorMap* m, bool is_f32, const void* base, int64_t P, int64_t rows, int box_rows) {
    if (!drv::api().tmap) throw Error(SG_E_CUDA, "cuTensorMapEncodeTiled unavailable");
    cuuint64_t dims[2] = {(cuuint64_t)P, (cuuint64_t)rows};
    cuuint64_t strides[1] = {(cuuint64_t)P * 4};
    cuuint32_t box[2] = {(cuuint32_t)P, (cuuint32_t)box_rows};
    cuuint32_t estr[2] = {1, 1};
    SG_CU(drv::api().tmap(m, is_f32 ? CU_TENSOR_MAP_DATA_TYPE_FLOAT32 : CU_TENSOR_MAP_DATA_TYPE_INT32, 2,
                          const_cast<void*>(base), dims, strides, box, estr, CU_TENSOR_MAP_INTERLEAVE_NONE,
                          CU_TENSOR_MAP_SWIZZLE_128B, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                          CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE));
}

int sm_count(int dev) {
    static std::map<int, int> cache;
    static std::mutex mu;
    std::lock_guard<std::mutex> lk(mu);
    auto it = cache.find(dev);
    if (it != cache.end()) return it->second;
    int n = 0;
    SG_RT(cudaDeviceGetAttribute(&n, cudaDevAttrMultiProcessorCount, dev));
    cache[dev] = n;
    return n;
}

// Launch one partition kernel over iterations [kb, ke) on `stream`.
int64_t launch(CompiledKernel& ck, int dev, const IoBinding& io, int64_t kb, int64_t ke, cudaStream_t stream,
               bool is_f32) {
    if (ke <= kb) return 0;
    ensure_module(ck, dev);
    std::vector<int64_t> v;
    for (auto p : io.in) v.push_back((int64_t)(uintptr_t)p);
    for (auto b : io.in_base) v.push_back(b);
    for (auto l : io.in_limit) v.push_back(l);
    for (auto p : io.out) v.push_back((int64_t)(uintptr_t)p);
    for (auto b : io.out_base) v.push_back(b);
    v.push_back(kb);
    v.push_back(ke);
    const KernelInfo& ki = ck.ki;
    if (ki.state_words > 0) {
        if ((int)ck.state.size() <= dev || !ck.state[dev]) throw Error(SG_E_CUDA, "internal: loop state not initialised");
        v.push_back((int64_t)(uintptr_t)ck.state[dev]);
    }
    if (ki.mode == 1 && ki.has_tma) {
        const char* in_row0 = (const char*)io.in[0] + (kb * ki.pin + ki.off_in - io.in_base[0]) * 4;
        char* out_row0 = (char*)io.out[0] + (kb * ki.pout + ki.off_out - io.out_base[0]) * 4;
        bool aligned = ((uintptr_t)in_row0 % 16 == 0) && ((uintptr_t)out_row0 % 16 == 0) && (ke - kb) < (1LL << 31);
        if (aligned) {
            alignas(64) CUtensorMap tin, tout;
            std::memset(&tin, 0, sizeof tin);
            std::memset(&tout, 0, sizeof tout);
            if (ki.tma_in == 1) encode_rows_map(&tin, is_f32, in_row0, ki.pin, ke - kb, ki.tile);
            if (ki.tma_out == 1) encode_rows_map(&tout, is_f32, out_row0, ki.pout, ke - kb, 32);
            int64_t tiles = (ke - kb + ki.tile - 1) / ki.tile;
            int64_t grid = std::min<int64_t>(tiles, (int64_t)sm_count(dev) * ck.max_blocks_per_sm[dev]);
            void* params[] = {v.data(), &tin, &tout};
            SG_CU(cuLaunchKernel(ck.fn[dev], (unsigned)grid, 1, 1, (unsigned)ki.threads, 1, 1, (unsigned)ki.smem,
                                 (CUstream)stream, params, nullptr));
            return 1;
        }
        int64_t tiles = (ke - kb + ki.tile_sync - 1) / ki.tile_sync;
        int64_t grid = std::min<int64_t>(tiles, (int64_t)sm_count(dev) * ck.max_blocks_sync[dev]);
        void* params[] = {v.data()};
        SG_CU(cuLaunchKernel(ck.fn_sync[dev], (unsigned)grid, 1, 1, (unsigned)ki.threads_sync, 1, 1,
                             (unsigned)ki.smem_sync, (CUstream)stream, params, nullptr));
        return 1;
    }
    if (ki.mode != 2) {  // register / bitslice / feedback-loop kernels
        int64_t tiles = (ke - kb + ki.tile - 1) / ki.tile;
        int64_t grid = std::min<int64_t>(tiles, (int64_t)sm_count(dev) * ck.max_blocks_per_sm[dev]);
        void* params[] = {v.data()};
        SG_CU(cuLaunchKernel(ck.fn[dev], (unsigned)grid, 1, 1, (unsigned)ki.threads, 1, 1, (unsigned)ki.smem,
                             (CUstream)stream, params, nullptr));
        return 1;
    }
    // staged kernels take [.., kb, ke, WR]: WR = iterations per tile for this launch (<= the compiled tile)
    v.push_back(ki.tile);
    const size_t IKB = v.size() - 3, IKE = v.size() - 2, IWR = v.size() - 1;
    const int64_t slots = (int64_t)sm_count(dev) * ck.max_blocks_per_sm[dev];
    // steady-state launch over [a, b) on `st` with `cap` CTA slots: fused kernels get a runtime tile that
    // makes every CTA process the same number of tiles (no straggler wave)
    auto main_launch = [&](int64_t a, int64_t b, cudaStream_t st, int64_t cap) {
        std::vector<int64_t> w = v;
        w[IKB] = a;
        w[IKE] = b;
        int64_t wr = ki.tile;
        const int64_t cnt = b - a;
        // opt-in (SG_RT_TILE=1): measured slower on FilterBank (0.217 vs 0.204 ms) -- the tile time is set by
        // rounds of NT-thread blocks per level (the cost model's W fills them), not by the iteration count
        if (ki.fused && std::getenv("SG_RT_TILE")) {
            const int64_t rounds = (cnt + cap * ki.tile - 1) / (cap * ki.tile);
            const int64_t even = (cnt + rounds * cap - 1) / (rounds * cap);
            if (even >= (ki.tile * 3) / 4 || rounds >= 4) wr = std::max<int64_t>(1, std::min<int64_t>(ki.tile, even));
        }
        w[IWR] = wr;
        const int64_t tiles = (cnt + wr - 1) / wr;
        const int64_t grid = std::max<int64_t>(1, std::min<int64_t>(tiles, cap));
        void* params[] = {w.data()};
        SG_CU(cuLaunchKernel(ck.fn[dev], (unsigned)grid, 1, 1, (unsigned)ki.threads, 1, 1, (unsigned)ki.smem,
                             (CUstream)st, params, nullptr));
    };
    if (!ki.name_start.empty() && kb < ki.ksafe) {
        // stream-start tiles (firings g < 0 must emit zeros): the guarded variant, compiled-tile sized
        const int64_t ks = std::min(ke, kb + ((ki.ksafe - kb + ki.tile - 1) / ki.tile) * ki.tile);
        const int64_t st_tiles = (ks - kb + ki.tile - 1) / ki.tile;
        std::vector<int64_t> v2 = v;
        v2[IKE] = ks;
        void* p2[] = {v2.data()};
        if (ks < ke && !std::getenv("SG_SERIAL_START")) {
            // on a side stream beside the steady-state kernel, which leaves them their CTA slots:
            // the start tiles no longer run alone before the main launch
            if ((int)ck.aux.size() <= dev) {
                ck.aux.resize(dev + 1, nullptr);
                ck.ev_fork.resize(dev + 1, nullptr);
                ck.ev_join.resize(dev + 1, nullptr);
            }
            if (!ck.aux[dev]) {
                SG_RT(cudaStreamCreateWithFlags(&ck.aux[dev], cudaStreamNonBlocking));
                SG_RT(cudaEventCreateWithFlags(&ck.ev_fork[dev], cudaEventDisableTiming));
                SG_RT(cudaEventCreateWithFlags(&ck.ev_join[dev], cudaEventDisableTiming));
            }
            SG_RT(cudaEventRecord(ck.ev_fork[dev], stream));
            SG_RT(cudaStreamWaitEvent(ck.aux[dev], ck.ev_fork[dev], 0));
            SG_CU(cuLaunchKernel(ck.fn_sync[dev], (unsigned)st_tiles, 1, 1, (unsigned)ki.threads, 1, 1, (unsigned)ki.smem,
                                 (CUstream)ck.aux[dev], p2, nullptr));
            SG_RT(cudaEventRecord(ck.ev_join[dev], ck.aux[dev]));
            main_launch(ks, ke, stream, std::max<int64_t>(1, slots - std::min<int64_t>(st_tiles, slots / 2)));
            SG_RT(cudaStreamWaitEvent(stream, ck.ev_join[dev], 0));
            return 2;
        }
        SG_CU(cuLaunchKernel(ck.fn_sync[dev], (unsigned)st_tiles, 1, 1, (unsigned)ki.threads, 1, 1, (unsigned)ki.smem,
                             (CUstream)stream, p2, nullptr));
        if (ke <= ks) return 1;
        main_launch(ks, ke, stream, slots);
        return 2;
    }
    main_launch(kb, ke, stream, slots);
    return 1;
}
}  // namespace

int64_t launch_kernel(CompiledKernel& ck, int dev, const IoBinding& io, int64_t kb, int64_t ke, cudaStream_t stream,
                      bool is_f32) {
    return launch(ck, dev, io, kb, ke, stream, is_f32);
}

void reset_state(CompiledKernel& ck, int dev, cudaStream_t stream) {
    if (ck.ki.state_words <= 0) return;
    if ((int)ck.state.size() <= dev) {
        ck.state.resize(dev + 1, nullptr);
        ck.state0.resize(dev + 1, nullptr);
    }
    const size_t bytes = (size_t)ck.ki.state_words * 4;
    if (!ck.state[dev]) {
        DevGuard dg(dev);
        SG_RT(cudaMalloc(&ck.state[dev], bytes));
        SG_RT(cudaMalloc(&ck.state0[dev], bytes));
        SG_RT(cudaMemcpy(ck.state0[dev], ck.ki.state_init.data(), bytes, cudaMemcpyHostToDevice));
    }
    DevGuard dg(dev);
    SG_RT(cudaMemcpyAsync(ck.state[dev], ck.state0[dev], bytes, cudaMemcpyDeviceToDevice, stream));
}

Plan::~Plan() {
    dist_release();
    for (auto e : host_ev) cudaEventDestroy(e);
    for (auto e : pipe_ev) cudaEventDestroy(e);
    if (host_in_stream) cudaStreamDestroy(host_in_stream);
    if (host_out_stream) cudaStreamDestroy(host_out_stream);
    for (auto& r : rings) {
        for (size_t i = 0; i < r.src_slots.size(); i++) {
            if (r.src_slots[i]) { cudaSetDevice(devices[r.src_gpu]); cudaFree(r.src_slots[i]); }
            if (r.dst_slots.size() > i && r.dst_slots[i] && r.dst_slots[i] != r.src_slots[i]) {
                cudaSetDevice(devices[r.dst_gpu]);
                cudaFree(r.dst_slots[i]);
            }
        }
        for (auto h : r.host_slots) if (h) cudaFreeHost(h);
        for (auto e : r.ev_copied) if (e) cudaEventDestroy(e);
        for (auto e : r.ev_consumed) if (e) cudaEventDestroy(e);
        for (auto e : r.ev_produced) if (e) cudaEventDestroy(e);
    }
    for (auto& g : gpus) {
        cudaSetDevice(g.dev);
        if (g.compute) cudaStreamDestroy(g.compute);
        if (g.copy) cudaStreamDestroy(g.copy);
        if (g.ev_start) cudaEventDestroy(g.ev_start);
        if (g.ev_done) cudaEventDestroy(g.ev_done);
    }
    if (user_ev) cudaEventDestroy(user_ev);
    if (host_in_dev) { cudaSetDevice(devices[input_gpu]); cudaFree(host_in_dev); }
    if (host_out_dev) { cudaSetDevice(devices[output_gpu]); cudaFree(host_out_dev); }
    if (host_stream) { cudaSetDevice(devices[input_gpu]); cudaStreamDestroy(host_stream); }
    for (auto& ck : kernels) {
        for (size_t d = 0; d < ck.mod.size(); d++)
            if (ck.mod[d]) { cudaSetDevice((int)d); drv::api().unload(ck.mod[d]); }
        for (size_t d = 0; d < ck.state.size(); d++) {
            if (ck.state[d]) { cudaSetDevice((int)d); cudaFree(ck.state[d]); }
            if (ck.state0[d]) { cudaSetDevice((int)d); cudaFree(ck.state0[d]); }
        }
        for (size_t d = 0; d < ck.aux.size(); d++) {
            if (!ck.aux[d]) continue;
            cudaSetDevice((int)d);
            cudaStreamDestroy(ck.aux[d]);
            cudaEventDestroy(ck.ev_fork[d]);
            cudaEventDestroy(ck.ev_join[d]);
        }
    }
}

void Plan::run(const void* in, int64_t n, void* out, cudaStream_t stream) {
    if (n <= 0) return;
    if (opts.plan_only) throw Error(SG_E_ARG, "plan was created with plan_only = 1");
    int ndev = 0;
    if (cudaGetDeviceCount(&ndev) != cudaSuccess || ndev <= 0) {
        cudaGetLastError();
        throw Error(SG_E_CUDA, "no CUDA device: the executor has no CPU fallback");
    }
    for (int d : devices)
        if (d >= ndev) throw Error(SG_E_CUDA, "plan maps a GPU to device " + std::to_string(d) + " but only " +
                                                  std::to_string(ndev) + " are visible");
    last_launches = 0;
    const int64_t n_in = flat.input_items(n);
    // ---- fast path: one partition on one GPU, launched on the caller's stream
    if (parts.size() == 1 && R == 1) {
        CompiledKernel& ck = kernels[0];
        DevGuard dg(devices[0]);
        IoBinding io;
        io.in = {in};
        io.in_base = {0};
        io.in_limit = {n_in};
        io.out = {out};
        io.out_base = {0};
        reset_state(ck, devices[0], stream);
        last_launches += launch(ck, devices[0], io, 0, n, stream, flat.dtype == SG_F32);
        return;
    }
    // ---- general path: fragments pipelined over partitions and GPUs
    int64_t F = fragment_size(*this, n);
    // the host pipeline (run_host) overlaps its copies fragment by fragment: about 8 of them
    const bool host_frag = pipe_hin && opts.iters_per_fragment <= 0;
    if (host_frag) F = std::max<int64_t>(1, std::min(F, (n + 7) / 8));
    // rings sized for a larger fragment serve a smaller one; without the host pipeline take their size
    if (rt_ready && rt_fragment >= F && !host_frag) F = std::min(rt_fragment, n);
    if (!rt_ready || rt_fragment < F) {
        // (re)allocate rings for fragment size F
        for (auto& r : rings) {
            for (size_t i = 0; i < r.src_slots.size(); i++) {
                cudaSetDevice(devices[r.src_gpu]);
                if (r.src_slots[i]) cudaFree(r.src_slots[i]);
                if (r.dst_slots[i] && r.dst_slots[i] != r.src_slots[i]) {
                    cudaSetDevice(devices[r.dst_gpu]);
                    cudaFree(r.dst_slots[i]);
                }
            }
            for (auto h : r.host_slots) if (h) cudaFreeHost(h);
            for (auto e : r.ev_copied) cudaEventDestroy(e);
            for (auto e : r.ev_consumed) cudaEventDestroy(e);
            for (auto e : r.ev_produced) cudaEventDestroy(e);
        }
        rings.clear();
        if (gpus.empty()) {
            gpus.resize(G);
            for (int g = 0; g < G; g++) {
                gpus[g].dev = devices[g];
                DevGuard dg(devices[g]);
                SG_RT(cudaStreamCreateWithFlags(&gpus[g].compute, cudaStreamNonBlocking));
                SG_RT(cudaStreamCreateWithFlags(&gpus[g].copy, cudaStreamNonBlocking));
                SG_RT(cudaEventCreateWithFlags(&gpus[g].ev_start, cudaEventDisableTiming));
                SG_RT(cudaEventCreateWithFlags(&gpus[g].ev_done, cudaEventDisableTiming));
            }
            // enable peer access between distinct physical devices
            for (int a = 0; a < G; a++)
                for (int b = 0; b < G; b++) {
                    if (devices[a] == devices[b]) continue;
                    int ok = 0;
                    cudaDeviceCanAccessPeer(&ok, devices[a], devices[b]);
                    if (ok) {
                        DevGuard dg(devices[a]);
                        cudaError_t e = cudaDeviceEnablePeerAccess(devices[b], 0);
                        if (e != cudaSuccess && e != cudaErrorPeerAccessAlreadyEnabled)
                            throw Error(SG_E_COMM, std::string("peer access: ") + cudaGetErrorString(e));
                        cudaGetLastError();
                    }
                }
        }
        // cut edges between partitions, one set of rings per replica group
        for (int grp = 0; grp < R; grp++)
        for (size_t ei = 0; ei < flat.edges.size(); ei++) {
            const Edge& ed = flat.edges[ei];
            if (ed.src < 0 || ed.dst < 0) continue;
            int ps = node_part[ed.src], pd = node_part[ed.dst];
            if (ps == pd || ring_rep[ei] != (int)ei) continue;  // members of a shared ring: below
            CutRing r;
            r.edge = (int)ei;
            r.group = grp;
            r.src_part = ps;
            r.dst_part = pd;
            for (size_t ej = 0; ej < flat.edges.size(); ej++)
                if (ring_rep[ej] == (int)ei && std::find(r.dst_parts.begin(), r.dst_parts.end(),
                                                         node_part[flat.edges[ej].dst]) == r.dst_parts.end())
                    r.dst_parts.push_back(node_part[flat.edges[ej].dst]);
            r.src_gpu = grp * Gs + part_gpu[ps];
            r.dst_gpu = grp * Gs + part_gpu[pd];
            cut_window((int)ei, r.lo, r.extra);
            r.per_iter = ed.per_iter;
            r.slot_items = r.per_iter * F + r.extra;
            for (int s = 0; s < ring_depth; s++) {
                void* p = nullptr;
                {
                    DevGuard dg(devices[r.src_gpu]);
                    SG_RT(cudaMalloc(&p, (size_t)r.slot_items * 4));
                }
                r.src_slots.push_back(p);
                void* q = p;
                if (r.dst_gpu != r.src_gpu) {
                    DevGuard dg(devices[r.dst_gpu]);
                    SG_RT(cudaMalloc(&q, (size_t)r.slot_items * 4));
                }
                r.dst_slots.push_back(q);
                void* h = nullptr;
                if (opts.transport == SG_TRANSPORT_HOST && r.dst_gpu != r.src_gpu)
                    SG_RT(cudaHostAlloc(&h, (size_t)r.slot_items * 4, cudaHostAllocPortable));
                r.host_slots.push_back(h);
                cudaEvent_t e1, e2, e3;
                {
                    DevGuard dg(devices[r.dst_gpu]);
                    SG_RT(cudaEventCreateWithFlags(&e2, cudaEventDisableTiming));
                }
                {
                    DevGuard dg(devices[r.src_gpu]);
                    SG_RT(cudaEventCreateWithFlags(&e1, cudaEventDisableTiming));
                    SG_RT(cudaEventCreateWithFlags(&e3, cudaEventDisableTiming));
                }
                r.ev_copied.push_back(e1);
                r.ev_consumed.push_back(e2);
                r.ev_produced.push_back(e3);
            }
            rings.push_back(std::move(r));
        }
        if (!user_ev) SG_RT(cudaEventCreateWithFlags(&user_ev, cudaEventDisableTiming));
        rt_fragment = F;
        rt_ready = true;
    }
    // per (group, partition): which rings feed it / leave it
    const size_t NP = parts.size();
    std::vector<std::vector<int>> ring_in(R * NP), ring_out(R * NP);
    for (size_t ri = 0; ri < rings.size(); ri++) {
        for (int dp : rings[ri].dst_parts) ring_in[rings[ri].group * NP + dp].push_back((int)ri);
        ring_out[rings[ri].group * NP + rings[ri].src_part].push_back((int)ri);
    }
    // order every GPU after the caller's stream
    SG_RT(cudaEventRecord(user_ev, stream));
    for (auto& g : gpus) {
        DevGuard dg(g.dev);
        SG_RT(cudaStreamWaitEvent(g.compute, user_ev, 0));
        SG_RT(cudaStreamWaitEvent(g.copy, user_ev, 0));
    }
    // feedback loops restart from their enqueued items (R = 1 for graphs with loops)
    for (size_t p = 0; p < parts.size(); p++)
        if (kernels[p].ki.state_words > 0) {
            GpuCtx& gc = gpus[part_gpu[p]];
            reset_state(kernels[p], gc.dev, gc.compute);
        }
    const int64_t nfrag = (n + F - 1) / F;
    // host pipeline (run_host): fragment fi's input prefix arrives on host_in_stream before the partition
    // reading the graph input runs it; its outputs leave on host_out_stream once the writing partition is done
    const bool pipe = pipe_hin != nullptr && R == 1;
    int64_t piped_in = 0;
    if (pipe)
        while ((int64_t)pipe_ev.size() < 2 * nfrag) {
            cudaEvent_t e;
            SG_RT(cudaEventCreateWithFlags(&e, cudaEventDisableTiming));
            pipe_ev.push_back(e);
        }
    for (int64_t fi = 0; fi < nfrag; fi++) {
        const int64_t ka = fi * F, kb = std::min(n, ka + F);
        // fragments dealt round-robin to the replica groups; rings are per group
        const int grp = (int)(fi % R);
        const int64_t fg = fi / R;
        const int slot = (int)(fg % ring_depth);
        if (pipe) {
            const int64_t need = flat.input_items(kb);
            if (need > piped_in) {
                DevGuard dg(devices[input_gpu]);
                SG_RT(cudaMemcpyAsync((char*)in + piped_in * 4, (const char*)pipe_hin + piped_in * 4,
                                      (size_t)(need - piped_in) * 4, cudaMemcpyHostToDevice, host_in_stream));
                piped_in = need;
            }
            SG_RT(cudaEventRecord(pipe_ev[2 * fi], host_in_stream));
        }
        for (int p : part_order) {
            CompiledKernel& ck = kernels[p];
            const int g = grp * Gs + part_gpu[p];
            const size_t gp = grp * NP + p;
            GpuCtx& gc = gpus[g];
            DevGuard dg(gc.dev);
            IoBinding io;
            bool writes_out = false;
            for (int e : ck.ki.in_edges) {
                if (flat.edges[e].src < 0) {  // graph input (resident on this GPU: input_gpu)
                    if (pipe) SG_RT(cudaStreamWaitEvent(gc.compute, pipe_ev[2 * fi], 0));
                    io.in.push_back(in);
                    io.in_base.push_back(0);
                    io.in_limit.push_back(n_in);
                    continue;
                }
                int ri = -1;
                for (int r : ring_in[gp]) if (rings[r].edge == ring_rep[e]) ri = r;
                if (ri < 0) throw Error(SG_E_PLAN, "internal: no ring for cut edge " + std::to_string(e));
                CutRing& r = rings[ri];
                if (r.src_gpu != r.dst_gpu) SG_RT(cudaStreamWaitEvent(gc.compute, r.ev_copied[slot], 0));
                io.in.push_back(r.dst_slots[slot]);
                io.in_base.push_back(ka * r.per_iter + r.lo);
                io.in_limit.push_back(r.slot_items);
            }
            for (int e : ck.ki.out_edges) {
                if (flat.edges[e].dst < 0) {
                    io.out.push_back(out);
                    io.out_base.push_back(0);
                    writes_out = true;
                    continue;
                }
                int ri = -1;
                for (int r : ring_out[gp]) if (rings[r].edge == ring_rep[e]) ri = r;
                if (ri < 0) throw Error(SG_E_PLAN, "internal: no ring for cut edge " + std::to_string(e));
                CutRing& r = rings[ri];
                // slot reuse: the copy (or the same-GPU consumer) of fragment fi - depth must be done
                if (fg >= ring_depth) {
                    if (r.src_gpu != r.dst_gpu) SG_RT(cudaStreamWaitEvent(gc.compute, r.ev_copied[slot], 0));
                    else SG_RT(cudaStreamWaitEvent(gc.compute, r.ev_consumed[slot], 0));
                }
                io.out.push_back(r.src_slots[slot]);
                io.out_base.push_back(ka * r.per_iter + r.lo);
            }
            last_launches += launch(ck, gc.dev, io, ka, kb, gc.compute, flat.dtype == SG_F32);
            if (pipe && writes_out) {
                SG_RT(cudaEventRecord(pipe_ev[2 * fi + 1], gc.compute));
                SG_RT(cudaStreamWaitEvent(host_out_stream, pipe_ev[2 * fi + 1], 0));
                const int64_t o0 = flat.output_items(ka), o1 = flat.output_items(kb);
                SG_RT(cudaMemcpyAsync((char*)pipe_hout + o0 * 4, (const char*)out + o0 * 4, (size_t)(o1 - o0) * 4,
                                      cudaMemcpyDeviceToHost, host_out_stream));
            }
            // consumed slots of incoming rings are free again
            for (int ri : ring_in[gp]) SG_RT(cudaEventRecord(rings[ri].ev_consumed[slot], gc.compute));
            // ship outgoing boundary streams to other GPUs (copy engine, P2P)
            for (int ri : ring_out[gp]) {
                CutRing& r = rings[ri];
                if (r.src_gpu == r.dst_gpu) continue;
                SG_RT(cudaEventRecord(r.ev_produced[slot], gc.compute));
                SG_RT(cudaStreamWaitEvent(gc.copy, r.ev_produced[slot], 0));
                if (fg >= ring_depth) SG_RT(cudaStreamWaitEvent(gc.copy, r.ev_consumed[slot], 0));
                int64_t items = r.per_iter * (kb - ka) + r.extra;
                const size_t bytes = (size_t)items * 4;
                if (opts.transport == SG_TRANSPORT_HOST) {
                    // host-staged pair, as in [7]: D2H into pinned memory, then H2D,
                    // in order on the producer's copy stream
                    SG_RT(cudaMemcpyAsync(r.host_slots[slot], r.src_slots[slot], bytes, cudaMemcpyDefault, gc.copy));
                    SG_RT(cudaMemcpyAsync(r.dst_slots[slot], r.host_slots[slot], bytes, cudaMemcpyDefault, gc.copy));
                } else if (opts.transport == SG_TRANSPORT_P2P || devices[r.src_gpu] != devices[r.dst_gpu]) {
                    SG_RT(cudaMemcpyPeerAsync(r.dst_slots[slot], devices[r.dst_gpu], r.src_slots[slot],
                                              devices[r.src_gpu], bytes, gc.copy));
                } else {
                    SG_RT(cudaMemcpyAsync(r.dst_slots[slot], r.src_slots[slot], bytes, cudaMemcpyDeviceToDevice,
                                          gc.copy));
                }
                SG_RT(cudaEventRecord(r.ev_copied[slot], gc.copy));
            }
        }
    }
    // join everything back onto the caller's stream
    for (auto& g : gpus) {
        DevGuard dg(g.dev);
        SG_RT(cudaEventRecord(g.ev_done, g.compute));
        SG_RT(cudaStreamWaitEvent(stream, g.ev_done, 0));
        SG_RT(cudaEventRecord(g.ev_start, g.copy));
        SG_RT(cudaStreamWaitEvent(stream, g.ev_start, 0));
    }
}

// HOST buffers in and out: H2D copy, run, D2H copy, synchronise (the end-to-end
// path a user without device memory takes).  Staging buffers are kept.
void Plan::run_host(const void* hin, int64_t n, void* hout) {
    if (n <= 0) return;
    int ndev = 0;
    if (cudaGetDeviceCount(&ndev) != cudaSuccess || ndev <= 0) {
        cudaGetLastError();
        throw Error(SG_E_CUDA, "no CUDA device: the executor has no CPU fallback");
    }
    const size_t bi = (size_t)flat.input_items(n) * 4, bo = (size_t)flat.output_items(n) * 4;
    const int din = devices[input_gpu], dout = devices[output_gpu];
    DevGuard dg(din);
    if (!host_stream) SG_RT(cudaStreamCreateWithFlags(&host_stream, cudaStreamNonBlocking));
    if (host_in_cap < bi) {
        if (host_in_dev) cudaFree(host_in_dev);
        host_in_dev = nullptr;
        SG_RT(cudaMalloc(&host_in_dev, bi));
        host_in_cap = bi;
    }
    if (host_out_cap < bo) {
        DevGuard d2(dout);
        if (host_out_dev) cudaFree(host_out_dev);
        host_out_dev = nullptr;
        SG_RT(cudaMalloc(&host_out_dev, bo));
        host_out_cap = bo;
    }
    // one partition (without a feedback loop): chunks of iterations pipelined over three streams, so
    // the host->device copy of chunk c+1, the kernel on chunk c and the device->host copy of chunk c-1
    // overlap (PCIe is full duplex; iterations are independent, and chunk c needs exactly the input
    // prefix input_items(end of c)).  Otherwise: copy in, run, copy out.
    const int NCH = std::getenv("SG_HOST_CHUNKS") ? std::atoi(std::getenv("SG_HOST_CHUNKS")) : 8;
    if (parts.size() == 1 && R == 1 && kernels[0].ki.state_words == 0 && NCH > 1 && n >= 4 * NCH) {
        if (!host_in_stream) {
            SG_RT(cudaStreamCreateWithFlags(&host_in_stream, cudaStreamNonBlocking));
            SG_RT(cudaStreamCreateWithFlags(&host_out_stream, cudaStreamNonBlocking));
        }
        while ((int)host_ev.size() < 2 * NCH + 1) {
            cudaEvent_t e;
            SG_RT(cudaEventCreateWithFlags(&e, cudaEventDisableTiming));
            host_ev.push_back(e);
        }
        CompiledKernel& ck = kernels[0];
        IoBinding io;
        io.in = {host_in_dev};
        io.in_base = {0};
        io.in_limit = {flat.input_items(n)};
        io.out = {host_out_dev};
        io.out_base = {0};
        reset_state(ck, din, host_stream);
        last_launches = 0;
        int64_t copied = 0;
        for (int c = 0; c < NCH; c++) {
            const int64_t ka = n * c / NCH, kb = n * (c + 1) / NCH;
            const int64_t need = flat.input_items(kb);
            if (need > copied) {
                SG_RT(cudaMemcpyAsync((char*)host_in_dev + copied * 4, (const char*)hin + copied * 4,
                                      (size_t)(need - copied) * 4, cudaMemcpyHostToDevice, host_in_stream));
                copied = need;
            }
            SG_RT(cudaEventRecord(host_ev[2 * c], host_in_stream));
            SG_RT(cudaStreamWaitEvent(host_stream, host_ev[2 * c], 0));
            last_launches += launch_kernel(ck, din, io, ka, kb, host_stream, flat.dtype == SG_F32);
            SG_RT(cudaEventRecord(host_ev[2 * c + 1], host_stream));
            SG_RT(cudaStreamWaitEvent(host_out_stream, host_ev[2 * c + 1], 0));
            const int64_t o0 = flat.output_items(ka), o1 = flat.output_items(kb);
            SG_RT(cudaMemcpyAsync((char*)hout + o0 * 4, (const char*)host_out_dev + o0 * 4, (size_t)(o1 - o0) * 4,
                                  cudaMemcpyDeviceToHost, host_out_stream));
        }
        SG_RT(cudaStreamSynchronize(host_out_stream));
        SG_RT(cudaStreamSynchronize(host_stream));
        return;
    }
    bool loops = false;
    for (auto& k : kernels) loops = loops || k.ki.state_words > 0;
    if (parts.size() > 1 && R == 1 && G == 1 && !loops && NCH > 1) {
        // several partitions: the fragment pipeline itself carries the copies (see run())
        if (!host_in_stream) {
            SG_RT(cudaStreamCreateWithFlags(&host_in_stream, cudaStreamNonBlocking));
            SG_RT(cudaStreamCreateWithFlags(&host_out_stream, cudaStreamNonBlocking));
        }
        pipe_hin = hin;
        pipe_hout = hout;
        try {
            run(host_in_dev, n, host_out_dev, host_stream);
        } catch (...) {
            pipe_hin = nullptr;
            pipe_hout = nullptr;
            throw;
        }
        pipe_hin = nullptr;
        pipe_hout = nullptr;
        SG_RT(cudaStreamSynchronize(host_out_stream));
        SG_RT(cudaStreamSynchronize(host_in_stream));
        SG_RT(cudaStreamSynchronize(host_stream));
        return;
    }
    SG_RT(cudaMemcpyAsync(host_in_dev, hin, bi, cudaMemcpyHostToDevice, host_stream));
    run(host_in_dev, n, host_out_dev, host_stream);
    SG_RT(cudaMemcpyAsync(hout, host_out_dev, bo, cudaMemcpyDeviceToHost, host_stream));
    SG_RT(cudaStreamSynchronize(host_stream));
}

}  // namespace sg

namespace sg {
// Time every partition's kernel alone over iterations [0, n) (the measured side
// of the PEE validation, Fig. 4.1 / PAPER.md:705-722).  Boundary streams come
// from zero-filled scratch windows of exactly the size sg_run's rings would
// hold for one fragment of n iterations; results in ns per iteration.
void Plan::profile_partitions(int64_t n, int reps, double* ns_per_iter) {
    if (n <= 0 || reps <= 0) throw Error(SG_E_ARG, "profile_partitions: n_iters and reps must be positive");
    if (opts.plan_only) throw Error(SG_E_ARG, "plan was created with plan_only = 1");
    int ndev = 0;
    if (cudaGetDeviceCount(&ndev) != cudaSuccess || ndev <= 0) {
        cudaGetLastError();
        throw Error(SG_E_CUDA, "no CUDA device: the executor has no CPU fallback");
    }
    const int64_t n_in = flat.input_items(n);
    for (size_t p = 0; p < parts.size(); p++) {
        CompiledKernel& ck = kernels[p];
        const int dev = devices[part_gpu[p]];
        DevGuard dg(dev);
        std::vector<void*> bufs;
        auto scratch = [&](int64_t items) {
            void* q = nullptr;
            SG_RT(cudaMalloc(&q, (size_t)std::max<int64_t>(items, 1) * 4));
            SG_RT(cudaMemset(q, 0, (size_t)std::max<int64_t>(items, 1) * 4));
            bufs.push_back(q);
            return q;
        };
        IoBinding io;
        for (int e : ck.ki.in_edges) {
            if (flat.edges[e].src < 0) {
                io.in.push_back(scratch(n_in));
                io.in_base.push_back(0);
                io.in_limit.push_back(n_in);
                continue;
            }
            int64_t lo, extra;
            edge_window(flat, e, lo, extra);
            int64_t items = flat.edges[e].per_iter * n + extra;
            io.in.push_back(scratch(items));
            io.in_base.push_back(lo);
            io.in_limit.push_back(items);
        }
        for (int e : ck.ki.out_edges) {
            if (flat.edges[e].dst < 0) {
                io.out.push_back(scratch(flat.output_items(n)));
                io.out_base.push_back(0);
                continue;
            }
            int64_t lo, extra;
            edge_window(flat, e, lo, extra);
            io.out.push_back(scratch(flat.edges[e].per_iter * n + extra));
            io.out_base.push_back(lo);
        }
        cudaStream_t s;
        cudaEvent_t e0, e1;
        SG_RT(cudaStreamCreateWithFlags(&s, cudaStreamNonBlocking));
        SG_RT(cudaEventCreate(&e0));
        SG_RT(cudaEventCreate(&e1));
        reset_state(ck, dev, s);
        launch(ck, dev, io, 0, n, s, flat.dtype == SG_F32);  // warm-up (module load, caches)
        SG_RT(cudaEventRecord(e0, s));
        for (int r = 0; r < reps; r++) {
            reset_state(ck, dev, s);  // feedback loops: every repetition starts from the stream start
            launch(ck, dev, io, 0, n, s, flat.dtype == SG_F32);
        }
        SG_RT(cudaEventRecord(e1, s));
        SG_RT(cudaEventSynchronize(e1));
        float ms = 0;
        SG_RT(cudaEventElapsedTime(&ms, e0, e1));
        ns_per_iter[p] = (double)ms * 1e6 / ((double)reps * (double)n);
        cudaEventDestroy(e0);
        cudaEventDestroy(e1);
        cudaStreamDestroy(s);
        for (void* q : bufs) cudaFree(q);
    }
}
}  // namespace sg
