// hrs_host.cuh -- host-side launch machinery of the hybrid radix sort, shared by the
// translation units that instantiate the kernels (hrs.cu: planner, C ABI, graph cache;
// inst_*.cu: the typed launch sequences, one unit per key width and key kind, compiled
// in parallel).  See include/hrs.h for the contract and hrs_device.cuh for the kernels.
#pragma once
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdint>
#include <cstdlib>
#include <cstring>
#include <mutex>
#include <type_traits>
#include <unordered_map>
#include <vector>

#include <nvtx3/nvToolsExt.h>

#include "hrs_device.cuh"

namespace hrs_host {
using namespace hrs;

extern thread_local int g_last_cuda;
extern thread_local uint64_t g_launches;

// ------------------------------------------------------------------ per-launch profiling (opt-in)
struct ProfRec {
    cudaEvent_t a, b;
    int kind, pass;
};
extern thread_local bool g_prof;
extern thread_local std::vector<ProfRec> g_prof_recs;
extern thread_local std::vector<cudaEvent_t> g_prof_pool;

inline cudaEvent_t prof_event() {
    if (!g_prof_pool.empty()) {
        cudaEvent_t e = g_prof_pool.back();
        g_prof_pool.pop_back();
        return e;
    }
    cudaEvent_t e = nullptr;
    cudaEventCreate(&e);
    return e;
}

// NVTX ranges around every launch, opt-in (HRS_NVTX=1 in the environment): named by kind
// (hist, classify, scatter, local, ...) so a timeline tool shows the pass structure
inline bool nvtx_enabled() {
    static const bool on = [] {
        const char *e = std::getenv("HRS_NVTX");
        return e && e[0] == '1';
    }();
    return on;
}
inline const char *kind_name(int kind) {
    static const char *const names[] = {"hrs:init", "hrs:hist", "hrs:scatter", "hrs:local", "hrs:copy", "hrs:classify"};
    return (kind >= 0 && kind < 6) ? names[kind] : "hrs:other";
}

// RAII bracket around one launch: counts it and, when profiling, records events
struct LaunchScope {
    cudaStream_t st;
    ProfRec rec;
    bool nvtx = false;
    LaunchScope(cudaStream_t s, int kind, int pass) : st(s) {
        ++g_launches;
        if (nvtx_enabled()) {
            nvtx = true;
            nvtxEventAttributes_t a;
            std::memset(&a, 0, sizeof(a));
            a.version = NVTX_VERSION;
            a.size = NVTX_EVENT_ATTRIB_STRUCT_SIZE;
            a.messageType = NVTX_MESSAGE_TYPE_ASCII;
            a.message.ascii = kind_name(kind);
            a.payloadType = NVTX_PAYLOAD_TYPE_INT32;
            a.payload.iValue = pass;
            nvtxRangePushEx(&a);
        }
        if (g_prof) {
            rec.kind = kind;
            rec.pass = pass;
            rec.a = prof_event();
            rec.b = prof_event();
            cudaEventRecord(rec.a, st);
        }
    }
    ~LaunchScope() {
        if (nvtx) nvtxRangePop();
        if (g_prof) {
            cudaEventRecord(rec.b, st);
            g_prof_recs.push_back(rec);
        }
    }
};

constexpr uint32_t DEFAULT_MT_DIV = 4;

// 32-bit-key scatter shape (overridable for experiments, micro/scatter_exp.py)
#ifndef HRS_SC_THREADS
#define HRS_SC_THREADS 256
#endif
#ifndef HRS_SC_KPT
#define HRS_SC_KPT 28  // measured on B200 (c2 uniform, both passes): 13 x 3 CTAs/SM 2.51 ms, 16 x 2 2.24, 20 x 2 2.15, 22 x 2 2.10, 32 x 1 2.41;
                       // one value buffer (HRS_SC_VSPLIT): 22 x 2 2.15, 26 x 2 2.09, 28 x 2 2.07 (AND-3 step 6.20 -> 6.00 ms)
#endif
#ifndef HRS_SC_NBUF
#define HRS_SC_NBUF 2
#endif
#ifndef HRS_SC_MINB
#define HRS_SC_MINB 2
#endif

// wider records (8-byte keys or values) scatter shape
#ifndef HRS_SC64_THREADS
#define HRS_SC64_THREADS 256
#endif
#ifndef HRS_SC64_KPT
#define HRS_SC64_KPT 15  // measured (c4 uniform / AND-3 step): 16 x 1 buffer 7.80 / 17.5 ms, 12 x 2 7.66 / 16.1, 22 x 1 7.52 / 17.2;
                         // one value buffer: 12 x 2 7.82 / 15.9, 14 x 2 7.56 / 15.6, 16 x 2 7.77 / 17.6;
                         // with the address table (PTR): 14 x 2 6.91, 15 x 2 6.86 (16 no longer fits two CTAs)
#endif
#ifndef HRS_SC64_MINB
#define HRS_SC64_MINB 2
#endif
#ifndef HRS_SC64_NBUF
#define HRS_SC64_NBUF 2
#endif

// ------------------------------------------------------------------ compile-time configurations

// scatter: THREADS x KPT records per tile (= the largest KPB); MINB resident CTAs per SM
template <int KB, int VB>
struct ScatterCfg {
    static constexpr bool SMALL = (KB == 4 && VB <= 4);
    static constexpr int THREADS = SMALL ? HRS_SC_THREADS : HRS_SC64_THREADS;
    static constexpr int KPT = SMALL ? HRS_SC_KPT : HRS_SC64_KPT;  // 256 x 28: two key buffers, one value buffer + the slot index for two CTAs per SM
    static constexpr int MINB = SMALL ? HRS_SC_MINB : HRS_SC64_MINB;
    static constexpr int NBUF = SMALL ? HRS_SC_NBUF : HRS_SC64_NBUF;
};
#ifndef HRS_HIST_THREADS
#define HRS_HIST_THREADS 256
#endif
constexpr int HIST_THREADS = HRS_HIST_THREADS;
constexpr int CLASSIFY_THREADS = 256;
constexpr uint32_t RANGE_MAX = 1024;  // >= SMs x resident scatter CTAs per SM
constexpr size_t SMEM_LIMIT = 227 * 1024;

template <int C>
struct LocalCfg;
template <> struct LocalCfg<0> { static constexpr int THREADS = 32, KPT = 4; };
template <> struct LocalCfg<1> { static constexpr int THREADS = 64, KPT = 4; };
template <> struct LocalCfg<2> { static constexpr int THREADS = 64, KPT = 8; };
template <> struct LocalCfg<3> { static constexpr int THREADS = 128, KPT = 8; };
#ifndef HRS_LC4_T
#define HRS_LC4_T 128
#endif
#ifndef HRS_LC4_K
#define HRS_LC4_K 16
#endif
template <> struct LocalCfg<4> { static constexpr int THREADS = HRS_LC4_T, KPT = HRS_LC4_K; };
static_assert(HRS_LC4_T * HRS_LC4_K >= 2048, "class 4 capacity");
template <> struct LocalCfg<5> { static constexpr int THREADS = 256, KPT = 16; };
template <> struct LocalCfg<6> { static constexpr int THREADS = 288, KPT = 16; };
template <> struct LocalCfg<7> { static constexpr int THREADS = 512, KPT = 16; };
// the counting local sort's CTA shape for classes 5 and 6 (same capacity as LocalCfg)
#ifndef HRS_LCC5_T
#define HRS_LCC5_T 256
#endif
#ifndef HRS_LCC5_K
#define HRS_LCC5_K 16
#endif
#ifndef HRS_LCC6_T
#define HRS_LCC6_T 256
#endif
#ifndef HRS_LCC6_K
#define HRS_LCC6_K 18
#endif
#ifndef HRS_LCC_OCC
#define HRS_LCC_OCC 4
#endif
#ifndef HRS_LCC5_OCC
#define HRS_LCC5_OCC HRS_LCC_OCC
#endif
#ifndef HRS_LCC6_OCC
#define HRS_LCC6_OCC HRS_LCC_OCC
#endif
template <int C>
struct LocalCntCfg : LocalCfg<C> {};
template <> struct LocalCntCfg<5> { static constexpr int THREADS = HRS_LCC5_T, KPT = HRS_LCC5_K; };
template <> struct LocalCntCfg<6> { static constexpr int THREADS = HRS_LCC6_T, KPT = HRS_LCC6_K; };
static_assert(HRS_LCC5_T * HRS_LCC5_K >= 4096 && HRS_LCC6_T * HRS_LCC6_K >= 4608, "class capacities");

// two-stage TMA prefetch where it fits next to a second resident CTA, else one stage
// two-stage TMA prefetch when three CTAs still fit per SM, else one stage; the
// register cap (launch bounds) is set for the occupancy the shared memory allows
template <typename K, typename V, int C, int WIDE = 0>
#ifndef HRS_WIDE_NSTAGE
#define HRS_WIDE_NSTAGE 1  // wide local sort of 8-byte keys: one staging buffer (measured, c4 AND-2 wide class 4: 5.61 -> 5.16 ms)
#endif
#ifndef HRS_WIDE_OCC
#define HRS_WIDE_OCC 6  // ... registers for six CTAs per SM (96, no spill) instead of three (167)
#endif
struct LocalStages {
    using LC = LocalCfg<C>;
    static constexpr size_t SM_BUDGET = 228 * 1024;  // shared memory per SM; 1 KB reserved per CTA
    static constexpr bool W64 = WIDE == 1 && sizeof(K) == 8;
    static constexpr int NSTAGE =
        (W64 && HRS_WIDE_NSTAGE) ? HRS_WIDE_NSTAGE
        : (3 * (LocalSmem<K, V, LC::THREADS, LC::KPT, 2, WIDE>::bytes + 1024) <= SM_BUDGET ? 2 : 1);
    static constexpr size_t bytes = LocalSmem<K, V, LC::THREADS, LC::KPT, NSTAGE, WIDE>::bytes;
    static constexpr bool fits = bytes <= SMEM_LIMIT && LocalSmem<K, V, LC::THREADS, LC::KPT, 1, 1>::bytes <= SMEM_LIMIT &&
                                 LocalSmem<K, V, LC::THREADS, LC::KPT, 1, 0>::bytes <= SMEM_LIMIT;
    static constexpr int by_smem = static_cast<int>(SM_BUDGET / (bytes + 1024));
    static constexpr int by_threads = 2048 / LC::THREADS;
    static constexpr int OCC0 = by_smem < by_threads ? by_smem : by_threads;
    static constexpr int OCC_CAP = W64 ? HRS_WIDE_OCC : 4;
    static constexpr int OCC = OCC0 < 1 ? 1 : (OCC0 > OCC_CAP ? OCC_CAP : OCC0);
};

// counting local sort (k_local_cnt) for the large classes: 2^15 counted values for 8-byte
// records, 2^14 for larger ones (shared memory for two or three CTAs per SM)
#ifndef HRS_LOCAL_CNT
#define HRS_LOCAL_CNT 1
#endif
#ifndef HRS_LC_NSTAGE
#define HRS_LC_NSTAGE 0  // 0: two stages when three CTAs still fit per SM
#endif
#ifndef HRS_LC_CB8
#define HRS_LC_CB8 14
#endif
constexpr int CNT_LO = 5, CNT_HI = 6;
template <typename K, typename V, int C, bool RECON>
struct LocalCntStages {
    using LC = LocalCntCfg<C>;
    static constexpr int VBYTES = HasVal<V>::value ? static_cast<int>(sizeof(V)) : 0;
    static constexpr int CB = static_cast<int>(sizeof(K)) + VBYTES <= 8 ? HRS_LC_CB8 : 14;
    static constexpr size_t SM_BUDGET = 228 * 1024;
    static constexpr int NSTAGE =
        HRS_LC_NSTAGE ? HRS_LC_NSTAGE
                      : (3 * (LocalCntSmem<K, V, LC::THREADS, LC::KPT, 2, CB, RECON>::bytes + 1024) <= SM_BUDGET ? 2 : 1);
    static constexpr size_t bytes = LocalCntSmem<K, V, LC::THREADS, LC::KPT, NSTAGE, CB, RECON>::bytes;
    static constexpr bool fits = HRS_LOCAL_CNT && LC::THREADS >= LC_SCAN && bytes <= SMEM_LIMIT;
    static constexpr int by_smem = static_cast<int>(SM_BUDGET / (bytes + 1024));
    static constexpr int by_threads = 2048 / LC::THREADS;
    static constexpr int OCC0 = by_smem < by_threads ? by_smem : by_threads;
    static constexpr int OCC_CAP = C == 5 ? HRS_LCC5_OCC : HRS_LCC6_OCC;
    static constexpr int OCC = OCC0 < 1 ? 1 : (OCC0 > OCC_CAP ? OCC_CAP : OCC0);
};

template <typename K, typename V>
constexpr int max_class_t() {
    return LocalStages<K, V, 7>::fits ? 7 : LocalStages<K, V, 6>::fits ? 6 : 5;
}

inline int max_class(int kb, int vb) {
    if (kb == 4) {
        if (vb == 0) return max_class_t<uint32_t, NoVal>();
        if (vb == 4) return max_class_t<uint32_t, uint32_t>();
        return max_class_t<uint32_t, unsigned long long>();
    }
    if (vb == 0) return max_class_t<unsigned long long, NoVal>();
    if (vb == 4) return max_class_t<unsigned long long, uint32_t>();
    return max_class_t<unsigned long long, unsigned long long>();
}

inline uint32_t max_kpb(int kb, int vb) {
    if (kb == 4 && vb <= 4) return ScatterCfg<4, 4>::THREADS * ScatterCfg<4, 4>::KPT;
    return ScatterCfg<8, 8>::THREADS * ScatterCfg<8, 8>::KPT;
}
inline uint32_t max_lt(int kb, int vb) { return class_capacity(max_class(kb, vb)); }

// ------------------------------------------------------------------ launch helpers

struct KernelInfo {
    int grid = 0;
};
extern std::mutex g_mu;
extern std::unordered_map<uint64_t, KernelInfo> g_kinfo;  // key: (device << 56) ^ fn pointer
extern std::unordered_map<int, int> g_dev_ok;  // device -> 1 ok / 0 not sm_100
extern std::unordered_map<int, int> g_dev_sms;

inline hrs_status cuda_fail(cudaError_t e) {
    g_last_cuda = static_cast<int>(e);
    return HRS_ERROR_CUDA;
}

inline hrs_status check_device(int *dev_out, int *sms_out) {
    int dev = 0;
    cudaError_t e = cudaGetDevice(&dev);
    if (e != cudaSuccess) return cuda_fail(e);
    std::lock_guard<std::mutex> lk(g_mu);
    auto it = g_dev_ok.find(dev);
    if (it == g_dev_ok.end()) {
        cudaDeviceProp prop;
        e = cudaGetDeviceProperties(&prop, dev);
        if (e != cudaSuccess) return cuda_fail(e);
        g_dev_ok[dev] = (prop.major == 10 && prop.minor == 0) ? 1 : 0;
        g_dev_sms[dev] = prop.multiProcessorCount;
        it = g_dev_ok.find(dev);
    }
    if (!it->second) return HRS_ERROR_NO_DEVICE;
    *dev_out = dev;
    *sms_out = g_dev_sms[dev];
    return HRS_SUCCESS;
}

// persistent grid = SMs x resident CTAs per SM (occupancy API), cached per kernel
template <typename F>
hrs_status grid_for(F *fn, int threads, size_t smem, int dev, int sms, int *grid) {
    const uint64_t key = (static_cast<uint64_t>(dev) << 56) ^ reinterpret_cast<uint64_t>(fn);
    {
        std::lock_guard<std::mutex> lk(g_mu);
        auto it = g_kinfo.find(key);
        if (it != g_kinfo.end()) {
            *grid = it->second.grid;
            return HRS_SUCCESS;
        }
    }
    cudaError_t e = cudaSuccess;
    if (smem > 48 * 1024) {
        e = cudaFuncSetAttribute(reinterpret_cast<const void *>(fn), cudaFuncAttributeMaxDynamicSharedMemorySize,
                                 static_cast<int>(smem));
        if (e != cudaSuccess) return cuda_fail(e);
    }
    int per_sm = 0;
    e = cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, reinterpret_cast<const void *>(fn), threads, smem);
    if (e != cudaSuccess) return cuda_fail(e);
    if (per_sm < 1) return cuda_fail(cudaErrorInvalidConfiguration);
    KernelInfo ki;
    ki.grid = per_sm * sms;
    {
        std::lock_guard<std::mutex> lk(g_mu);
        g_kinfo[key] = ki;
    }
    *grid = ki.grid;
    return HRS_SUCCESS;
}

// launch with programmatic stream serialization (PDL); kernels call pdl_wait() first
template <typename... KArgs, typename... Args>
void launch_pdl(void (*fn)(KArgs...), dim3 grid, dim3 block, size_t smem, cudaStream_t st, Args &&...args) {
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = grid;
    cfg.blockDim = block;
    cfg.dynamicSmemBytes = smem;
    cfg.stream = st;
    cudaLaunchAttribute attr[1];
    attr[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    attr[0].val.programmaticStreamSerializationAllowed = 1;
    cfg.attrs = attr;
    cfg.numAttrs = 1;
    cudaLaunchKernelEx(&cfg, fn, std::forward<Args>(args)...);
}

inline hrs_status last_launch() {
    cudaError_t e = cudaGetLastError();
    if (e != cudaSuccess) return cuda_fail(e);
    return HRS_SUCCESS;
}

// ------------------------------------------------------------------ conditional graph capture (small sorts)
//
// While a small sort's launch sequence is captured into a CUDA graph (hrs.cu, via_graph),
// g_gx points at this context: every pass after the first becomes a conditional IF node
// (nested: pass p + 1 inside pass p) whose value the previous pass's scatter sets, and the
// local-sort launches IF nodes whose values one small kernel sets from the list counts.
// A replay then runs only the launches that have work (constant launches per
// pass -- but a pass with no bucket needs none).  Any API failure abandons the capture (the
// caller falls back to a plain capture).
struct GraphCtx {
    std::vector<cudaStream_t> pool;  // capture streams of the nested bodies
    size_t depth = 0;
    bool ok = true;
    bool graph_of(cudaStream_t st, cudaGraph_t *g, const cudaGraphNode_t **deps, size_t *nd) {
        cudaStreamCaptureStatus cs = cudaStreamCaptureStatusNone;
        if (cudaStreamGetCaptureInfo(st, &cs, nullptr, g, deps, nd) != cudaSuccess ||
            cs != cudaStreamCaptureStatusActive)
            return ok = false;
        return true;
    }
    bool handle(cudaStream_t st, cudaGraphConditionalHandle *h) {
        cudaGraph_t g;
        const cudaGraphNode_t *deps;
        size_t nd;
        if (!graph_of(st, &g, &deps, &nd)) return false;
        if (cudaGraphConditionalHandleCreate(h, g, 0, cudaGraphCondAssignDefault) != cudaSuccess) return ok = false;
        return true;
    }
    // IF(h) after the work captured so far on st; returns the stream capturing its body
    cudaStream_t if_begin(cudaStream_t st, cudaGraphConditionalHandle h) {
        cudaGraph_t g;
        const cudaGraphNode_t *deps;
        size_t nd;
        if (!graph_of(st, &g, &deps, &nd)) return nullptr;
        cudaGraphNodeParams np = {cudaGraphNodeTypeConditional};
        np.conditional.handle = h;
        np.conditional.type = cudaGraphCondTypeIf;
        np.conditional.size = 1;
        cudaGraphNode_t node;
        if (cudaGraphAddNode(&node, g, deps, nd, &np) != cudaSuccess) return ok = false, nullptr;
        if (cudaStreamUpdateCaptureDependencies(st, &node, 1, cudaStreamSetCaptureDependencies) != cudaSuccess)
            return ok = false, nullptr;
        if (depth == pool.size()) {
            cudaStream_t ns = nullptr;
            if (cudaStreamCreateWithFlags(&ns, cudaStreamNonBlocking) != cudaSuccess) return ok = false, nullptr;
            pool.push_back(ns);
        }
        cudaStream_t bs = pool[depth++];
        if (cudaStreamBeginCaptureToGraph(bs, np.conditional.phGraph_out[0], nullptr, nullptr, 0,
                                          cudaStreamCaptureModeThreadLocal) != cudaSuccess)
            return ok = false, nullptr;
        return bs;
    }
    void if_end(cudaStream_t bs) {
        cudaGraph_t g = nullptr;
        if (cudaStreamEndCapture(bs, &g) != cudaSuccess) ok = false;
        --depth;
    }
};
extern thread_local GraphCtx *g_gx;

// side streams for the independent local-sort launches (per device, created on first use)
// and per-thread fork/join events (hrs.cu); HRS_FORK=0 launches them in order on the
// caller's stream instead
cudaStream_t side_stream(int dev, int i);
cudaEvent_t fork_event(int i);
inline bool fork_enabled() {
    static const bool on = [] {
        const char *e = std::getenv("HRS_FORK");
        return !(e && e[0] == '0');
    }();
    return on;
}

// ------------------------------------------------------------------ plan + temp layout

enum Mode { MODE_SORT = 0, MODE_HIST = 1, MODE_PARTITION = 2 };

struct Plan {
    uint64_t n = 0;
    int kb = 4, vb = 0;
    int begin = 0, end = 0;
    int D = 0;
    int lo[HRS_MAX_PASSES] = {0}, hi[HRS_MAX_PASSES] = {0};
    uint32_t lt = 0, mt = 0, kpb = 0;
    int single_class = -1;
    bool counting = false;
    uint32_t tile_cap = 0, bucket_cap = 0;
    uint32_t local_cap[HRS_NUM_CLASSES] = {0};
    uint32_t range_cap = 0;  // CTAs of the hist/scatter grid the temp layout allows
    size_t off_auxk = 0, off_auxv = 0, off_buckets[2] = {0, 0}, off_tot[2] = {0, 0}, off_subrel = 0,
           off_seg_last = 0, off_seg_meta = 0, off_carry = 0, off_tiles = 0, off_tile_pref = 0,
           off_local[HRS_NUM_CLASSES] = {0}, off_local_wide[HRS_NUM_CLASSES] = {0}, off_local_fb2 = 0, total = 0;
    uint32_t local_wide_cap[HRS_NUM_CLASSES] = {0}, local_fb2_cap = 0;
    int wide_top = 0;
    int force_redo = 0;  // HRS_FLAG_FORCE_REDO (tuning flags or the HRS_FORCE_REDO environment variable)
    int kind = 0;        // hrs_key_kind of the keys (signed / float: the bijection fused into the kernels)
    bool dst = false;    // hrs_partition_pass_to: the scatter writes each digit to its own window
    size_t off_dst = 0;  //   (tables in temp: 256 digit offsets, MAX_WINDOWS key / value windows)
};
constexpr int MAX_WINDOWS = 64;

// HRS_FORCE_REDO=1 in the environment ORs HRS_FLAG_FORCE_REDO into every call (include/hrs.h)
inline uint32_t env_flags() {
    static const uint32_t f = [] {
        const char *e = std::getenv("HRS_FORCE_REDO");
        return (e && e[0] == '1') ? HRS_FLAG_FORCE_REDO : 0u;
    }();
    return f;
}

inline size_t align_up(size_t x, size_t a) { return (x + a - 1) / a * a; }

inline hrs_status make_plan(Plan &pl, uint64_t n, int kb, int vb, int begin, int end, const hrs_tuning *tu, Mode mode) {
    pl.n = n;
    pl.kb = kb;
    pl.vb = vb;
    pl.begin = begin;
    pl.end = end;
    hrs_tuning t;
    t.local_threshold = 8192;
    t.merge_threshold = 8192 / DEFAULT_MT_DIV;
    t.keys_per_tile = max_kpb(kb, vb);
    t.local_classes = 0;
    t.flags = 0;
    if (tu) {
        if (tu->local_threshold) t.local_threshold = tu->local_threshold;
        if (tu->merge_threshold) t.merge_threshold = tu->merge_threshold;
        else if (tu->local_threshold) t.merge_threshold = std::max<uint32_t>(1, t.local_threshold / DEFAULT_MT_DIV);
        if (tu->keys_per_tile) t.keys_per_tile = tu->keys_per_tile;
        t.local_classes = tu->local_classes;
        t.flags = tu->flags;
    }
    if (t.flags & ~HRS_FLAG_FORCE_REDO) return HRS_ERROR_INVALID_VALUE;
    pl.force_redo = ((t.flags | env_flags()) & HRS_FLAG_FORCE_REDO) ? 1 : 0;
    if (t.local_threshold < 1 || t.local_threshold > max_lt(kb, vb)) return HRS_ERROR_INVALID_VALUE;
    if (t.merge_threshold < 1 || t.merge_threshold > t.local_threshold) return HRS_ERROR_INVALID_VALUE;
    if (t.keys_per_tile < 1 || t.keys_per_tile > max_kpb(kb, vb)) return HRS_ERROR_INVALID_VALUE;
    if (t.local_classes > 1) return HRS_ERROR_INVALID_VALUE;
    pl.lt = t.local_threshold;
    pl.mt = t.merge_threshold;
    pl.kpb = t.keys_per_tile;
    pl.single_class = t.local_classes ? size_class_of(pl.lt) : -1;

    // digit plan: 8-bit digits aligned to end_bit, most-significant first (reading #3)
    pl.D = 0;
    for (int h = end; h > begin; h -= 8) {
        pl.hi[pl.D] = h;
        pl.lo[pl.D] = std::max(begin, h - 8);
        ++pl.D;
    }
    if (mode != MODE_SORT) pl.D = 1;
    pl.counting = (mode != MODE_SORT) ? (n > 0) : (n > pl.lt && begin < end);

    // analytical bounds: I1 buckets <= n/∂ˆ, I4 tiles <= n/KPB + n/∂ˆ
    const uint64_t lt = pl.lt, kpb = pl.kpb;
    uint64_t tiles = n / kpb + n / lt + 2;
    uint64_t buckets = n / lt + 2;
    if (mode != MODE_SORT) {
        tiles = n / kpb + 2;
        buckets = 2;
    }
    pl.tile_cap = static_cast<uint32_t>(std::min<uint64_t>(tiles, 0xFFFFFFFFull));
    pl.bucket_cap = static_cast<uint32_t>(std::min<uint64_t>(buckets, 0xFFFFFFFFull));
    // local lists: class c >= 1 entries hold > 64 * 2^c records; class 0 bounded by the
    // merge rule (I3: any two neighbouring groups hold >= ∂ records)
    for (int c = 0; c < HRS_NUM_CLASSES; ++c) {
        uint64_t cap = 0;
        if (mode == MODE_SORT) {
            if (pl.single_class >= 0) {
                cap = c == pl.single_class ? std::min<uint64_t>(n, 2 * n / pl.mt + 2 * pl.D * (n / lt + 1)) + 2 : 0;
            } else if (c == 0) {
                cap = std::min<uint64_t>(n, 2 * n / pl.mt + 2 * pl.D * (n / lt + 1)) + 2;
            } else if (class_capacity(c - 1) < pl.lt) {
                cap = n / (class_capacity(c - 1) + 1ull) + 2;  // entries of class c hold > capacity(c - 1)
            }
            if (!pl.counting) cap = (c == (pl.single_class >= 0 ? pl.single_class : size_class_of((uint32_t)std::max<uint64_t>(n, 1)))) ? 1 : 0;
        }
        pl.local_cap[c] = static_cast<uint32_t>(std::min<uint64_t>(cap, 0xFFFFFFFFull));
    }

    // temp layout
    size_t off = align_up(sizeof(Ctl), 256);
    const bool need_aux = (mode == MODE_SORT) && pl.counting && pl.D >= 2;
    pl.off_auxk = off;
    if (need_aux) off = align_up(off + n * kb, 256);
    pl.off_auxv = off;
    if (need_aux && vb) off = align_up(off + n * vb, 256);
    for (int i = 0; i < 2; ++i) {
        pl.off_buckets[i] = off;
        off = align_up(off + sizeof(Bucket) * static_cast<size_t>(pl.bucket_cap), 256);
        pl.off_tot[i] = off;
        off = align_up(off + sizeof(uint32_t) * RADIX * static_cast<size_t>(pl.bucket_cap), 256);
    }
    pl.range_cap = std::min<uint32_t>(RANGE_MAX, pl.tile_cap);
    pl.off_seg_last = off;
    off = align_up(off + sizeof(uint32_t) * RADIX * static_cast<size_t>(pl.range_cap), 256);
    pl.off_carry = off;
    off = align_up(off + sizeof(uint32_t) * RADIX * static_cast<size_t>(pl.range_cap), 256);
    pl.off_seg_meta = off;
    off = align_up(off + sizeof(RangeMeta) * static_cast<size_t>(pl.range_cap), 256);
    pl.off_tiles = off;
    off = align_up(off + sizeof(TileDesc) * static_cast<size_t>(pl.tile_cap), 256);
    pl.off_tile_pref = off;
    off = align_up(off + sizeof(uint32_t) * RADIX * static_cast<size_t>(pl.tile_cap), 256);
    pl.off_subrel = off;
    off = align_up(off + sizeof(uint32_t) * RADIX * static_cast<size_t>(pl.bucket_cap), 256);
    uint64_t fb = 0;
    for (int c = 0; c < HRS_NUM_CLASSES; ++c) {
        pl.off_local[c] = off;
        off = align_up(off + sizeof(LocalEntry) * static_cast<size_t>(pl.local_cap[c]), 256);
        fb += pl.local_cap[c];
    }
    // entries of more than 19 sort bits whose top bits tie in long runs go to the wide
    // local sort, to the list of the wide configuration of their size class (every entry
    // of the single-configuration ablation to its one class)
    (void)fb;
    pl.wide_top = max_class(kb, vb);
    uint64_t wcap[HRS_NUM_CLASSES] = {0};
    for (int c = 0; c < HRS_NUM_CLASSES; ++c)
        wcap[pl.single_class >= 0 ? pl.single_class : wide_cfg(c, pl.wide_top, kb == 8)] += pl.local_cap[c];
    for (int c = 0; c < HRS_NUM_CLASSES; ++c) {
        pl.local_wide_cap[c] = static_cast<uint32_t>(std::min<uint64_t>(wcap[c], 0xFFFFFFFFull));
        pl.off_local_wide[c] = off;
        off = align_up(off + sizeof(LocalEntry) * static_cast<size_t>(pl.local_wide_cap[c]), 256);
    }
    // entries the counting local sort (classes CNT_LO..CNT_HI) hands to the narrow one
    uint64_t fb2 = 0;
    for (int c = CNT_LO; c <= CNT_HI; ++c) fb2 += pl.local_cap[c];
    pl.local_fb2_cap = static_cast<uint32_t>(std::min<uint64_t>(fb2, 0xFFFFFFFFull));
    pl.off_local_fb2 = off;
    off = align_up(off + sizeof(LocalEntry) * static_cast<size_t>(pl.local_fb2_cap), 256);
    pl.off_dst = off;
    if (mode == MODE_PARTITION) off = align_up(off + sizeof(uint64_t) * (RADIX + 2 * MAX_WINDOWS), 256);
    pl.total = off;
    return HRS_SUCCESS;
}

inline bool overlap(const void *a, size_t na, const void *b, size_t nb) {
    if (!a || !b || !na || !nb) return false;
    const uintptr_t x = reinterpret_cast<uintptr_t>(a), y = reinterpret_cast<uintptr_t>(b);
    return x < y + nb && y < x + na;
}

template <typename P>
P *at(void *base, size_t off) {
    return reinterpret_cast<P *>(static_cast<unsigned char *>(base) + off);
}

// ------------------------------------------------------------------ typed launch sequences

template <typename K, typename V, bool TY>
struct Runner {
    static constexpr int KB = sizeof(K);
    static constexpr int VB = HasVal<V>::value ? sizeof(V) : 0;
    // histogram staging = one scatter tile (the largest KPB of this key/value type)
    static constexpr int HIST_CAP = ScatterCfg<KB, VB>::THREADS * ScatterCfg<KB, VB>::KPT;
    using SC = ScatterCfg<KB, (VB == 0 ? 4 : VB)>;

    static hrs_status init(const Plan &pl, void *temp, cudaStream_t st, int sms, int root_class, int counting,
                           const uint64_t *grouped_hist = nullptr) {
        InitParams ip;
        ip.grouped_hist = grouped_hist;
        ip.grouped_radix = 1u << (pl.hi[0] - pl.lo[0]);
        ip.ctl = at<Ctl>(temp, 0);
        ip.buckets = at<Bucket>(temp, pl.off_buckets[1]);
        ip.tot = at<uint32_t>(temp, pl.off_tot[1]);
        ip.root_local = root_class >= 0 ? at<LocalEntry>(temp, pl.off_local[root_class]) : nullptr;
        ip.root_class = root_class;
        ip.n = pl.n;
        ip.kpb = pl.kpb;
        ip.counting = counting;
        ip.end_bit = pl.end;
        ip.key_bytes = pl.kb;
        ip.value_bytes = pl.vb;
        LaunchScope ls(st, 0, 0);
        launch_pdl(k_init, dim3(1), dim3(256), 0, st, ip);
        return last_launch();
    }

    // the hist / classify grid of a pass (CTAs = contiguous tile runs): the hist
    // kernel's persistent grid, capped by the temp layout
    static hrs_status range_grid(const Plan &pl, int dev, int sms, uint32_t *G) {
        auto fn = k_hist<K, HIST_THREADS, HIST_CAP, TY>;
        int grid = 0;
        hrs_status s = grid_for(fn, HIST_THREADS, 0, dev, sms, &grid);
        if (s) return s;
        *G = std::min<uint32_t>(static_cast<uint32_t>(grid), pl.range_cap);
        return HRS_SUCCESS;
    }

    // the three buffers a bucket can live in (Bucket::src): the input, the aux buffer in
    // temp and the output
    struct Bufs {
        const void *k[3];
        const void *v[3];
    };
    static Bufs bufs(const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout) {
        Bufs b;
        b.k[SRC_IN] = kin;
        b.k[SRC_AUX] = at<void>(temp, pl.off_auxk);
        b.k[SRC_OUT] = kout;
        b.v[SRC_IN] = vin;
        b.v[SRC_AUX] = VB ? at<void>(temp, pl.off_auxv) : nullptr;
        b.v[SRC_OUT] = vout;
        return b;
    }

    static hrs_status hist(const Plan &pl, void *temp, cudaStream_t st, int dev, int sms, int p, const Bufs &bf,
                           uint32_t G) {
        HistParams hp;
        hp.n = pl.n;
        for (int i = 0; i < 3; ++i) hp.src_keys[i] = bf.k[i];
        hp.kind = pl.kind;
        hp.p = p;
        hp.lo = pl.lo[p - 1];
        hp.mask = (1u << (pl.hi[p - 1] - pl.lo[p - 1])) - 1u;
        hp.kpb = pl.kpb;
        hp.buckets = at<Bucket>(temp, pl.off_buckets[p & 1]);
        hp.tot = at<uint32_t>(temp, pl.off_tot[p & 1]);
        hp.seg_last = at<uint32_t>(temp, pl.off_seg_last);
        hp.seg_meta = at<RangeMeta>(temp, pl.off_seg_meta);
        hp.tiles = at<TileDesc>(temp, pl.off_tiles);
        hp.tile_pref = at<uint32_t>(temp, pl.off_tile_pref);
        hp.ctl = at<Ctl>(temp, 0);
        auto fn = k_hist<K, HIST_THREADS, HIST_CAP, TY>;
        LaunchScope ls(st, 1, p);
        launch_pdl(fn, dim3(G), dim3(HIST_THREADS), 0, st, hp);
        return last_launch();
    }

    static hrs_status classify(const Plan &pl, void *temp, cudaStream_t st, int dev, int sms, int p,
                               uint16_t src_code, uint64_t *out_hist, uint64_t *out_offsets, bool last, uint32_t G) {
        ClassifyParams cp;
        std::memset(&cp, 0, sizeof(cp));
        cp.p = p;
        cp.last = last ? 1 : 0;
        cp.lo = pl.lo[p - 1];
        cp.width = pl.hi[p - 1] - pl.lo[p - 1];
        cp.buckets = at<Bucket>(temp, pl.off_buckets[p & 1]);
        cp.tot = at<uint32_t>(temp, pl.off_tot[p & 1]);
        cp.tot_next = at<uint32_t>(temp, pl.off_tot[(p + 1) & 1]);
        cp.next_buckets = at<Bucket>(temp, pl.off_buckets[(p + 1) & 1]);
        cp.sub_rel = at<uint32_t>(temp, pl.off_subrel);
        cp.seg_last = at<uint32_t>(temp, pl.off_seg_last);
        cp.seg_meta = at<RangeMeta>(temp, pl.off_seg_meta);
        cp.carry = at<uint32_t>(temp, pl.off_carry);
        cp.ranges = G;
        cp.ctl = at<Ctl>(temp, 0);
        for (int c = 0; c < HRS_NUM_CLASSES; ++c) {
            cp.local[c] = at<LocalEntry>(temp, pl.off_local[c]);
            cp.local_cap[c] = pl.local_cap[c];
        }
        cp.tile_cap = pl.tile_cap;
        cp.bucket_cap = pl.bucket_cap;
        cp.lt = pl.lt;
        cp.mt = pl.mt;
        cp.kpb = pl.kpb;
        cp.single_class = pl.single_class;
        cp.src_code = src_code;
        cp.out_hist = out_hist;
        cp.out_offsets = out_offsets;
        auto fn = k_classify<CLASSIFY_THREADS>;
        int grid = 0;
        hrs_status s = grid_for(fn, CLASSIFY_THREADS, 0, dev, sms, &grid);
        if (s) return s;
        // one block per bucket (up to the resident limit) plus the carry block
        grid = static_cast<int>(std::min<uint64_t>(grid, std::max<uint64_t>(pl.bucket_cap, 1))) + CARRY_CTAS;
        LaunchScope ls(st, 5, p);
        launch_pdl(fn, dim3(grid), dim3(CLASSIFY_THREADS), 0, st, cp);
        return last_launch();
    }

    static hrs_status scatter(const Plan &pl, void *temp, cudaStream_t st, int dev, int sms, int p, const Bufs &bf,
                              void *kout, void *vout, uint32_t G, const cudaGraphConditionalHandle *next = nullptr) {
        ScatterParams sp;
        std::memset(&sp, 0, sizeof(sp));
        if (next) {
            sp.next_cond = *next;
            sp.has_next_cond = 1;
        }
        sp.n = pl.n;
        for (int i = 0; i < 3; ++i) {
            sp.src_keys[i] = bf.k[i];
            sp.src_vals[i] = bf.v[i];
        }
        sp.keys_out = kout;
        sp.vals_out = vout;
        sp.p = p;
        sp.lo = pl.lo[p - 1];
        sp.mask = (1u << (pl.hi[p - 1] - pl.lo[p - 1])) - 1u;
        sp.buckets = at<Bucket>(temp, pl.off_buckets[p & 1]);
        sp.sub_rel = at<uint32_t>(temp, pl.off_subrel);
        sp.carry = at<uint32_t>(temp, pl.off_carry);
        sp.tiles = at<TileDesc>(temp, pl.off_tiles);
        sp.tile_pref = at<uint32_t>(temp, pl.off_tile_pref);
        sp.ctl = at<Ctl>(temp, 0);
        sp.force_redo = pl.force_redo;
        sp.kind = pl.kind;
        sp.final_pass = p == pl.D ? 1 : 0;
        if constexpr (!TY) {
            if (pl.dst) {  // hrs_partition_pass_to: every digit to its own window
                sp.dst_off = at<unsigned long long>(temp, pl.off_dst);
                sp.dst_kwin = sp.dst_off + RADIX;
                sp.dst_vwin = sp.dst_kwin + MAX_WINDOWS;
                auto fd = k_scatter<K, V, SC::THREADS, SC::KPT, SC::MINB, SC::NBUF, false, true>;
                const size_t smd = ScatterSmem<K, V, SC::THREADS, SC::KPT, SC::NBUF, true>::bytes;
                int gd = 0;
                hrs_status sd = grid_for(fd, SC::THREADS, smd, dev, sms, &gd);
                if (sd) return sd;
                LaunchScope ls(st, 2, p);
                launch_pdl(fd, dim3(gd), dim3(SC::THREADS), smd, st, sp);
                return last_launch();
            }
        }
        auto fn = k_scatter<K, V, SC::THREADS, SC::KPT, SC::MINB, SC::NBUF, TY>;
        const size_t smem = ScatterSmem<K, V, SC::THREADS, SC::KPT, SC::NBUF>::bytes;
        int grid = 0;
        hrs_status s = grid_for(fn, SC::THREADS, smem, dev, sms, &grid);
        if (s) return s;
        (void)G;
        LaunchScope ls(st, 2, p);
        launch_pdl(fn, dim3(grid), dim3(SC::THREADS), smem, st, sp);
        return last_launch();
    }

    // which list a local launch sorts: its class list, or a hand-off list
    enum LocalList { LIST_CLASS = 0, LIST_FB = 1, LIST_FB2 = 2 };

    static void local_params(LocalParams &lp, const Plan &pl, void *temp, const void *kin, void *kout,
                             const void *vin, void *vout) {
        lp.n = pl.n;
        lp.src_keys[SRC_IN] = kin;
        lp.src_keys[SRC_AUX] = at<void>(temp, pl.off_auxk);
        lp.src_keys[SRC_OUT] = kout;
        lp.src_vals[SRC_IN] = vin;
        lp.src_vals[SRC_AUX] = VB ? at<void>(temp, pl.off_auxv) : nullptr;
        lp.src_vals[SRC_OUT] = vout;
        lp.keys_out = kout;
        lp.vals_out = vout;
        lp.begin_bit = pl.begin;
        lp.force_redo = pl.force_redo;
        lp.redo = &at<Ctl>(temp, 0)->redo;
        lp.kind = pl.kind;
    }

    // the counting local sort of class C; hands what it does not take to LIST_FB2
    template <int C, bool RECON>
    static hrs_status local_cnt_variant(const Plan &pl, void *temp, cudaStream_t st, int dev, int sms,
                                        const void *kin, void *kout, const void *vin, void *vout) {
        using LST = LocalCntStages<K, V, C, RECON>;
        if constexpr (!LST::fits) {
            return HRS_ERROR_INVALID_VALUE;
        } else {
            using LC = LocalCntCfg<C>;
            LocalParams lp;
            local_params(lp, pl, temp, kin, kout, vin, vout);
            Ctl *ctl = at<Ctl>(temp, 0);
            lp.list = at<LocalEntry>(temp, pl.off_local[C]);
            lp.count = &ctl->nlocal[C];
            lp.fb_list = at<LocalEntry>(temp, pl.off_local_fb2);
            lp.fb_count = &ctl->nlocal_fb2;
            lp.fb_cap = pl.local_fb2_cap;
            auto fn = k_local_cnt<K, V, LC::THREADS, LC::KPT, LST::NSTAGE, LST::OCC, LST::CB, RECON, TY>;
            int grid = 0;
            hrs_status s = grid_for(fn, LC::THREADS, LST::bytes, dev, sms, &grid);
            if (s) return s;
            grid = static_cast<int>(std::min<uint64_t>(grid, std::max<uint32_t>(pl.local_cap[C], 1)));
            LaunchScope ls(st, 3, C);
            launch_pdl(fn, dim3(grid), dim3(LC::THREADS), LST::bytes, st, lp);
            return last_launch();
        }
    }

    // the counting variant serves classes CNT_LO..CNT_HI when it fits this key/value type
    static constexpr bool cnt_ok(int c) {
        return c >= CNT_LO && c <= CNT_HI && c <= max_class_t<K, V>() &&
               (c == 5 ? LocalCntStages<K, V, 5, false>::fits && (KB != 4 || LocalCntStages<K, V, 5, true>::fits)
                       : LocalCntStages<K, V, 6, false>::fits && (KB != 4 || LocalCntStages<K, V, 6, true>::fits));
    }
    static bool recon(const Plan &pl) { return KB == 4 && pl.begin == 0 && pl.end == 32; }

    template <int C, int WIDE>
    static hrs_status local_variant(const Plan &pl, void *temp, cudaStream_t st, int dev, int sms, const void *kin,
                                    void *kout, const void *vin, void *vout, int which = LIST_CLASS) {
        using LST = LocalStages<K, V, C, WIDE>;
        if constexpr (!LST::fits) {
            return HRS_ERROR_INVALID_VALUE;
        } else {
            using LC = LocalCfg<C>;
            LocalParams lp;
            local_params(lp, pl, temp, kin, kout, vin, vout);
            Ctl *ctl = at<Ctl>(temp, 0);
            lp.fb_list = nullptr;
            lp.fb_count = nullptr;
            lp.fb_cap = 0;
            for (int c = 0; c < HRS_NUM_CLASSES; ++c) {
                lp.wide_list[c] = at<LocalEntry>(temp, pl.off_local_wide[c]);
                lp.wide_cap[c] = pl.local_wide_cap[c];
            }
            lp.wide_count = ctl->nlocal_wide;
            lp.wide_single = pl.single_class;
            lp.wide_top = pl.wide_top;
            uint32_t cap = pl.local_cap[C];
            if (which == LIST_FB) {  // the wide variant of configuration C sorts what was handed to it
                lp.list = lp.wide_list[C];
                lp.count = &ctl->nlocal_wide[C];
                cap = pl.local_wide_cap[C];
            } else if (which == LIST_FB2) {  // what the counting variant handed over
                lp.list = at<LocalEntry>(temp, pl.off_local_fb2);
                lp.count = &ctl->nlocal_fb2;
                cap = pl.local_fb2_cap;
            } else {
                lp.list = at<LocalEntry>(temp, pl.off_local[C]);
                lp.count = &ctl->nlocal[C];
            }
            auto fn = k_local<K, V, LC::THREADS, LC::KPT, LST::NSTAGE, LST::OCC, WIDE, TY>;
            int grid = 0;
            hrs_status s = grid_for(fn, LC::THREADS, LST::bytes, dev, sms, &grid);
            if (s) return s;
            grid = static_cast<int>(std::min<uint64_t>(grid, std::max<uint32_t>(cap, 1)));
            LaunchScope ls(st, 3, which == LIST_FB ? 10 + C : which == LIST_FB2 ? 9 : C);
            launch_pdl(fn, dim3(grid), dim3(LC::THREADS), LST::bytes, st, lp);
            return last_launch();
        }
    }

    template <int C>
    static hrs_status local_one(const Plan &pl, void *temp, cudaStream_t st, int dev, int sms, const void *kin,
                                void *kout, const void *vin, void *vout) {
        if constexpr (cnt_ok(C)) {
            if (pl.single_class < 0) {  // (the single-configuration ablation keeps k_local)
                if constexpr (KB == 4)
                    if (recon(pl)) return local_cnt_variant<C, true>(pl, temp, st, dev, sms, kin, kout, vin, vout);
                return local_cnt_variant<C, false>(pl, temp, st, dev, sms, kin, kout, vin, vout);
            }
        }
        // full-range sorts of 32-bit keys rebuild the keys from the composites: every key
        // bit above a bucket's sorted bits is then a digit it was partitioned on, common
        // to the bucket (with end_bit < 32 the bits above end_bit vary and are carried)
        if (KB == 4 && pl.begin == 0 && pl.end == 32)
            return local_variant<C, 2>(pl, temp, st, dev, sms, kin, kout, vin, vout);
        return local_variant<C, 0>(pl, temp, st, dev, sms, kin, kout, vin, vout);
    }

    // the local-sort launches fork onto side streams for small sorts only: there their
    // launch latencies dominate (c1 2^20 keys: 0.091 -> 0.084 ms); at 2^28 the overlapping
    // kernels only compete (c2 +0.7 %)
    static int fork_dev(const Plan &pl, int dev) { return pl.n <= (1ull << 22) ? dev : -1; }

    // launch(i, stream) for every i: directly, or -- under a conditional graph capture --
    // each inside IF(the list `what[i]` is non-empty), one k_set_conds in front
    template <typename F>
    static hrs_status cond_group(cudaStream_t st, void *temp, const int *what, int n, F &&launch, int dev = -1) {
        GraphCtx *gx = g_gx;
        if (!gx) {
            if (n > 1 && dev >= 0 && fork_enabled()) {
                // independent launches (different lists, disjoint outputs): one side stream
                // each, joined back into st -- their launch latencies overlap (small sorts)
                // and their tails overlap (large ones)
                cudaEvent_t e0 = fork_event(0);
                if (cudaEventRecord(e0, st) != cudaSuccess) return cuda_fail(cudaGetLastError());
                for (int i = 0; i < n; ++i) {
                    cudaStream_t si = side_stream(dev, i);
                    if (!si || cudaStreamWaitEvent(si, e0, 0) != cudaSuccess) return cuda_fail(cudaGetLastError());
                    const hrs_status s = launch(i, si);
                    if (s) return s;
                    cudaEvent_t ei = fork_event(1 + i);
                    if (cudaEventRecord(ei, si) != cudaSuccess || cudaStreamWaitEvent(st, ei, 0) != cudaSuccess)
                        return cuda_fail(cudaGetLastError());
                }
                return HRS_SUCCESS;
            }
            for (int i = 0; i < n; ++i) {
                const hrs_status s = launch(i, st);
                if (s) return s;
            }
            return HRS_SUCCESS;
        }
        for (int i0 = 0; i0 < n; i0 += MAX_CONDS) {
            const int m = std::min(n - i0, MAX_CONDS);
            CondSet cs;
            std::memset(&cs, 0, sizeof(cs));
            cs.n = m;
            cs.ctl = at<Ctl>(temp, 0);
            for (int i = 0; i < m; ++i) {
                if (!gx->handle(st, &cs.h[i])) return HRS_ERROR_CUDA;
                cs.what[i] = static_cast<uint32_t>(what[i0 + i]);
            }
            {
                LaunchScope ls(st, 4, 0);
                launch_pdl(k_set_conds, dim3(1), dim3(32), 0, st, cs);
            }
            hrs_status s = last_launch();
            if (s) return s;
            for (int i = 0; i < m; ++i) {
                cudaStream_t bs = gx->if_begin(st, cs.h[i]);
                if (!bs) return HRS_ERROR_CUDA;
                s = launch(i0 + i, bs);
                gx->if_end(bs);
                if (s) return s;
                if (!gx->ok) return HRS_ERROR_CUDA;
            }
        }
        return HRS_SUCCESS;
    }

    static hrs_status wide_one(int c, const Plan &pl, void *temp, cudaStream_t st, int dev, int sms, const void *kin,
                               void *kout, const void *vin, void *vout) {
        switch (c) {
            case 0: return local_variant<0, 1>(pl, temp, st, dev, sms, kin, kout, vin, vout, LIST_FB);
            case 1: return local_variant<1, 1>(pl, temp, st, dev, sms, kin, kout, vin, vout, LIST_FB);
            case 2: return local_variant<2, 1>(pl, temp, st, dev, sms, kin, kout, vin, vout, LIST_FB);
            case 3: return local_variant<3, 1>(pl, temp, st, dev, sms, kin, kout, vin, vout, LIST_FB);
            case 4: return local_variant<4, 1>(pl, temp, st, dev, sms, kin, kout, vin, vout, LIST_FB);
            case 5: return local_variant<5, 1>(pl, temp, st, dev, sms, kin, kout, vin, vout, LIST_FB);
            case 6: return local_variant<6, 1>(pl, temp, st, dev, sms, kin, kout, vin, vout, LIST_FB);
            case 7: return local_variant<7, 1>(pl, temp, st, dev, sms, kin, kout, vin, vout, LIST_FB);
        }
        return HRS_ERROR_INVALID_VALUE;
    }

    // the wide launches for whatever the narrow ones handed over, one per wide
    // configuration (wide_cfg: 1024, 2048, [4096, 4608 for 64-bit keys,] largest); only needed when more than 19 bits
    // can remain to sort
    static hrs_status local_wide(const Plan &pl, void *temp, cudaStream_t st, int dev, int sms, const void *kin,
                                 void *kout, const void *vin, void *vout) {
        if (pl.end - pl.begin <= 19) return HRS_SUCCESS;  // every entry fits a narrow composite
        int cfg[8], n = 0;
        if (pl.single_class >= 0) {
            cfg[n++] = pl.single_class;
        } else {
            const int cmax = size_class_of(pl.lt);
            cfg[n++] = 3;
            if (cmax >= 4) cfg[n++] = 4;
            if (HRS_WIDE_MID && KB == 8 && cmax >= 5 && max_class_t<K, V>() > 5) cfg[n++] = 5;
            if (HRS_WIDE_MID && KB == 8 && cmax >= 6 && max_class_t<K, V>() > 6) cfg[n++] = 6;
            if (cmax >= 5) cfg[n++] = max_class_t<K, V>() == 7 ? 7 : 6;
        }
        int what[8];
        for (int i = 0; i < n; ++i) what[i] = 16 + cfg[i];
        return cond_group(st, temp, what, n, [&](int i, cudaStream_t s2) {
            return wide_one(cfg[i], pl, temp, s2, dev, sms, kin, kout, vin, vout);
        }, fork_dev(pl, dev));
    }

    // the narrow k_local over the entries the counting variant handed over (sizes up to
    // the capacity of class CNT_HI); launched whenever a counting launch was
    static hrs_status local_fb2(const Plan &pl, void *temp, cudaStream_t st, int dev, int sms, const void *kin,
                                void *kout, const void *vin, void *vout) {
        constexpr int CF = max_class_t<K, V>() < CNT_HI ? max_class_t<K, V>() : CNT_HI;
        if (recon(pl)) return local_variant<CF, 2>(pl, temp, st, dev, sms, kin, kout, vin, vout, LIST_FB2);
        return local_variant<CF, 0>(pl, temp, st, dev, sms, kin, kout, vin, vout, LIST_FB2);
    }

    static hrs_status local(const Plan &pl, void *temp, cudaStream_t st, int dev, int sms, int c, const void *kin,
                            void *kout, const void *vin, void *vout) {
        switch (c) {
            case 0: return local_one<0>(pl, temp, st, dev, sms, kin, kout, vin, vout);
            case 1: return local_one<1>(pl, temp, st, dev, sms, kin, kout, vin, vout);
            case 2: return local_one<2>(pl, temp, st, dev, sms, kin, kout, vin, vout);
            case 3: return local_one<3>(pl, temp, st, dev, sms, kin, kout, vin, vout);
            case 4: return local_one<4>(pl, temp, st, dev, sms, kin, kout, vin, vout);
            case 5: return local_one<5>(pl, temp, st, dev, sms, kin, kout, vin, vout);
            case 6: return local_one<6>(pl, temp, st, dev, sms, kin, kout, vin, vout);
            case 7: return local_one<7>(pl, temp, st, dev, sms, kin, kout, vin, vout);
        }
        return HRS_ERROR_INVALID_VALUE;
    }

    // grouped: the input is already grouped by its first digit (hrs_sort_grouped) with the
    // device histogram `grouped`; pass 1's partition is skipped (X_1 = the input)
    static hrs_status sort(const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout,
                           cudaStream_t st, int dev, int sms, const uint64_t *grouped = nullptr) {
        hrs_status s;
        const int root_class =
            pl.counting ? -1
                        : (pl.single_class >= 0 ? pl.single_class
                                                : size_class_of((uint32_t)std::max<uint64_t>(pl.n, 1)));
        // a grouped input on a single digit is already the stable sort: one copy
        const bool copy_only = grouped && pl.counting && pl.D == 1;
        if ((s = init(pl, temp, st, sms, pl.n > 0 && pl.begin < pl.end ? root_class : -1, pl.counting ? 1 : 0,
                      pl.counting && !copy_only ? grouped : nullptr)))
            return s;
        if (pl.n == 0) return HRS_SUCCESS;
        if (pl.begin == pl.end || copy_only) {
            using VC = typename std::conditional<VB == 8, uint64_t, uint32_t>::type;
            const int grid = static_cast<int>(std::min<uint64_t>((pl.n + 255) / 256, static_cast<uint64_t>(sms) * 8));
            {
                LaunchScope ls(st, 4, 0);
                k_copy<K><<<grid, 256, 0, st>>>(static_cast<const K *>(kin), static_cast<K *>(kout), pl.n);
            }
            if ((s = last_launch())) return s;
            if (VB) {
                LaunchScope ls(st, 4, 0);
                k_copy<VC><<<grid, 256, 0, st>>>(static_cast<const VC *>(vin), static_cast<VC *>(vout), pl.n);
                if ((s = last_launch())) return s;
            }
            return HRS_SUCCESS;
        }
        void *auxk = at<void>(temp, pl.off_auxk);
        void *auxv = VB ? at<void>(temp, pl.off_auxv) : nullptr;
        if (pl.counting) {
            uint32_t G = 0;
            if ((s = range_grid(pl, dev, sms, &G))) return s;
            const Bufs bf = bufs(pl, temp, kin, kout, vin, vout);
            GraphCtx *gx = g_gx;
            cudaStream_t cur = st;  // (inside the nested conditional bodies under graph capture)
            cudaStream_t opened[HRS_MAX_PASSES + 1];
            int nopen = 0;
            for (int p = 1; p <= pl.D; ++p) {
                const bool to_out = ((pl.D - p) % 2) == 0;
                void *yk = to_out ? kout : auxk;
                void *yv = to_out ? vout : auxv;
                if (p == 1 && grouped) {
                    // the partition on digit 1 is given: classify its histogram (no per-CTA
                    // ranges), the sub-buckets stay in the input (X_1 = in)
                    if ((s = classify(pl, temp, cur, dev, sms, 1, SRC_IN, nullptr, nullptr, false, 0))) return s;
                    continue;
                }
                if ((s = hist(pl, temp, cur, dev, sms, p, bf, G))) return s;
                if ((s = classify(pl, temp, cur, dev, sms, p, to_out ? SRC_OUT : SRC_AUX, nullptr, nullptr,
                                  p == pl.D, G)))
                    return s;
                cudaGraphConditionalHandle hn;
                const bool cond = gx && p < pl.D;
                if (cond && !gx->handle(cur, &hn)) return HRS_ERROR_CUDA;
                if ((s = scatter(pl, temp, cur, dev, sms, p, bf, yk, yv, G, cond ? &hn : nullptr))) return s;
                if (cond) {  // pass p + 1 runs iff it has buckets
                    cur = gx->if_begin(cur, hn);
                    if (!cur) return HRS_ERROR_CUDA;
                    opened[nopen++] = cur;
                }
            }
            while (nopen > 0) gx->if_end(opened[--nopen]);
            if (gx && !gx->ok) return HRS_ERROR_CUDA;
            const int cmax = pl.single_class >= 0 ? pl.single_class : size_class_of(pl.lt);
            const int c0 = pl.single_class >= 0 ? pl.single_class : 0;
            int what[HRS_NUM_CLASSES];
            bool cnt = false;
            for (int c = c0; c <= cmax; ++c) {
                what[c - c0] = c;
                cnt = cnt || (pl.single_class < 0 && cnt_ok(c));
            }
            if ((s = cond_group(st, temp, what, cmax - c0 + 1, [&](int i, cudaStream_t s2) {
                     return local(pl, temp, s2, dev, sms, c0 + i, kin, kout, vin, vout);
                 }, fork_dev(pl, dev))))
                return s;
            const int w8 = 8;
            if (cnt && (s = cond_group(st, temp, &w8, 1, [&](int, cudaStream_t s2) {
                            return local_fb2(pl, temp, s2, dev, sms, kin, kout, vin, vout);
                        })))
                return s;
        } else {
            if ((s = local(pl, temp, st, dev, sms, root_class, kin, kout, vin, vout))) return s;
            if (pl.single_class < 0 && cnt_ok(root_class) &&
                (s = local_fb2(pl, temp, st, dev, sms, kin, kout, vin, vout)))
                return s;
        }
        if ((s = local_wide(pl, temp, st, dev, sms, kin, kout, vin, vout))) return s;
        return HRS_SUCCESS;
    }

    static hrs_status building_block(const Plan &pl, void *temp, const void *kin, void *kout, const void *vin,
                                     void *vout, uint64_t *out_hist, uint64_t *out_offsets, bool do_scatter,
                                     cudaStream_t st, int dev, int sms) {
        hrs_status s;
        if ((s = init(pl, temp, st, sms, -1, pl.n > 0 ? 1 : 0))) return s;
        const int r = 1 << (pl.hi[0] - pl.lo[0]);
        if (pl.n == 0) {
            uint64_t *p = out_hist ? out_hist : out_offsets;
            if (p) {
                LaunchScope ls(st, 4, 0);
                k_fill_u64<<<1, 256, 0, st>>>(p, static_cast<uint64_t>(r) + (out_hist ? 0 : 1), 0);
                return last_launch();
            }
            return HRS_SUCCESS;
        }
        uint32_t G = 0;
        if ((s = range_grid(pl, dev, sms, &G))) return s;
        const Bufs bf = bufs(pl, temp, kin, kout, vin, vout);
        if ((s = hist(pl, temp, st, dev, sms, 1, bf, G))) return s;
        if ((s = classify(pl, temp, st, dev, sms, 1, SRC_OUT, out_hist, out_offsets, true, G))) return s;
        if (do_scatter && (s = scatter(pl, temp, st, dev, sms, 1, bf, kout, vout, G))) return s;
        return HRS_SUCCESS;
    }
};

template <typename K, typename V, bool TY>
hrs_status run_sort(const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout,
                    cudaStream_t st, int dev, int sms, const uint64_t *grouped) {
    return Runner<K, V, TY>::sort(pl, temp, kin, kout, vin, vout, st, dev, sms, grouped);
}

template <typename K, typename V>
hrs_status run_block(const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout,
                     uint64_t *h, uint64_t *o, bool sc, cudaStream_t st, int dev, int sms) {
    return Runner<K, V, false>::building_block(pl, temp, kin, kout, vin, vout, h, o, sc, st, dev, sms);
}


inline bool aligned(const void *p, size_t a) { return (reinterpret_cast<uintptr_t>(p) % a) == 0; }

// per-unit entry points (inst_*.cu): one launch sequence for key width KB, typed (TY) or not
hrs_status sort_k4(int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout,
                   cudaStream_t st, int dev, int sms, const uint64_t *grouped);
hrs_status sort_k8(int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout,
                   cudaStream_t st, int dev, int sms, const uint64_t *grouped);
hrs_status sort_k4t(int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout,
                    cudaStream_t st, int dev, int sms, const uint64_t *grouped);
hrs_status sort_k8t(int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout,
                    cudaStream_t st, int dev, int sms, const uint64_t *grouped);
hrs_status block_k4(int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout,
                    uint64_t *h, uint64_t *o, bool sc, cudaStream_t st, int dev, int sms);
hrs_status block_k8(int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin, void *vout,
                    uint64_t *h, uint64_t *o, bool sc, cudaStream_t st, int dev, int sms);

}  // namespace hrs_host
