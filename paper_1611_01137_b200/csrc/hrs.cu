// hrs.cu -- host planner, launch dispatch and C ABI of the hybrid radix sort.
//
// See include/hrs.h for the contract and hrs_device.cuh for the kernels.  The
// host side only validates arguments, computes the digit plan and the temp
// layout from the analytical bounds of P:815-874 (I1-I4, M1-M5), and enqueues a
// constant number of launches per pass.  It never reads device memory
// during a sort.
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdint>
#include <cstdlib>
#include <cstring>
#include <mutex>
#include <type_traits>
#include <unordered_map>
#include <vector>

#include "hrs_device.cuh"

using namespace hrs;
#include "hrs_host.cuh"

using namespace hrs;
using namespace hrs_host;

namespace hrs_host {
thread_local int g_last_cuda = 0;
thread_local uint64_t g_launches = 0;
thread_local bool g_prof = false;
thread_local std::vector<ProfRec> g_prof_recs;
thread_local std::vector<cudaEvent_t> g_prof_pool;
std::mutex g_mu;
std::unordered_map<uint64_t, KernelInfo> g_kinfo;
std::unordered_map<int, int> g_dev_ok;
std::unordered_map<int, int> g_dev_sms;
thread_local GraphCtx *g_gx = nullptr;

cudaStream_t side_stream(int dev, int i) {
    // per thread: a stream being captured into one thread's graph must not receive another
    // thread's launches
    thread_local std::unordered_map<int, std::vector<cudaStream_t>> streams;
    auto &v = streams[dev];
    while (static_cast<int>(v.size()) <= i) {
        cudaStream_t s = nullptr;
        if (cudaStreamCreateWithFlags(&s, cudaStreamNonBlocking) != cudaSuccess) return nullptr;
        v.push_back(s);
    }
    return v[i];
}

cudaEvent_t fork_event(int i) {
    thread_local std::vector<cudaEvent_t> ev;
    while (static_cast<int>(ev.size()) <= i) {
        cudaEvent_t e = nullptr;
        if (cudaEventCreateWithFlags(&e, cudaEventDisableTiming) != cudaSuccess) return nullptr;
        ev.push_back(e);
    }
    return ev[i];
}
}  // namespace hrs_host

namespace {

hrs_status sort_dispatch(int kb, int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin,
                         void *vout, cudaStream_t st, int dev, int sms, const uint64_t *grouped = nullptr) {
    if (pl.kind != 0)
        return kb == 4 ? sort_k4t(vb, pl, temp, kin, kout, vin, vout, st, dev, sms, grouped)
                       : sort_k8t(vb, pl, temp, kin, kout, vin, vout, st, dev, sms, grouped);
    return kb == 4 ? sort_k4(vb, pl, temp, kin, kout, vin, vout, st, dev, sms, grouped)
                   : sort_k8(vb, pl, temp, kin, kout, vin, vout, st, dev, sms, grouped);
}

hrs_status block_dispatch(int kb, int vb, const Plan &pl, void *temp, const void *kin, void *kout, const void *vin,
                          void *vout, uint64_t *h, uint64_t *o, bool sc, cudaStream_t st, int dev, int sms) {
    return kb == 4 ? block_k4(vb, pl, temp, kin, kout, vin, vout, h, o, sc, st, dev, sms)
                   : block_k8(vb, pl, temp, kin, kout, vin, vout, h, o, sc, st, dev, sms);
}


// ------------------------------------------------------------------ graph cache (small sorts)
//
// A sort enqueues a fixed sequence of ~25 launches whatever its size; below ~2^22
// records the host's launch submissions take longer than the GPU work.  The second
// call with identical arguments (sizes, bits, tuning, every pointer, device) captures
// the sequence on a private stream into a CUDA graph (programmatic-dependent-launch
// edges included), and that and every later such call replays it with one
// cudaGraphLaunch into the caller's stream.  (The first call runs directly, which
// also fills the per-kernel grid cache outside any capture.)  HRS_GRAPHS=0 disables it;
// per-launch profiling bypasses it.
#ifndef HRS_GRAPH_MAX_N
#define HRS_GRAPH_MAX_N (1ull << 22)
#endif
struct GraphKey {
    uint64_t v[16];
    bool operator==(const GraphKey &o) const { return std::memcmp(v, o.v, sizeof(v)) == 0; }
};
struct GraphKeyHash {
    size_t operator()(const GraphKey &k) const {
        uint64_t h = 0x9E3779B97F4A7C15ull;
        for (uint64_t x : k.v) h = (h ^ x) * 0xBF58476D1CE4E5B9ull;
        return static_cast<size_t>(h ^ (h >> 31));
    }
};
struct GraphEntry {
    cudaGraphExec_t exec = nullptr;  // null: seen once, not captured yet
    uint64_t launches = 0;
    uint64_t stamp = 0;
};
std::mutex g_gmu;
std::unordered_map<GraphKey, GraphEntry, GraphKeyHash> g_graphs;
std::unordered_map<int, cudaStream_t> g_capture_stream;
uint64_t g_gstamp = 0;
constexpr size_t GRAPH_CACHE_MAX = 64;

std::unordered_map<int, GraphCtx> g_gctx;  // conditional-capture streams per device

// Conditional capture is opt-in (HRS_GRAPH_COND=1): measured on B200, c1 (2^20 keys) replays
// in 0.186 ms with conditional nodes against 0.101 ms as a plain graph -- an IF node costs
// more than the empty launches it skips (profiles/r02_c1_cond_graph.txt)
bool cond_graphs_enabled() {
    static const bool on = [] {
        const char *e = std::getenv("HRS_GRAPH_COND");
        return e && e[0] == '1';
    }();
    return on;
}

bool graphs_enabled() {
    static const bool on = [] {
        const char *e = std::getenv("HRS_GRAPHS");
        return !(e && e[0] == '0');
    }();
    return on;
}

// Runs `run(stream)` through the graph cache; returns false when the cache does not
// apply (then the caller launches directly).
template <typename F>
bool via_graph(const GraphKey &key, cudaStream_t stream, int dev, hrs_status *out, F &&run) {
    std::lock_guard<std::mutex> lk(g_gmu);
    auto it = g_graphs.find(key);
    if (it == g_graphs.end()) {
        if (g_graphs.size() >= GRAPH_CACHE_MAX) {  // evict the least recently used
            auto lru = g_graphs.begin();
            for (auto j = g_graphs.begin(); j != g_graphs.end(); ++j)
                if (j->second.stamp < lru->second.stamp) lru = j;
            if (lru->second.exec) cudaGraphExecDestroy(lru->second.exec);
            g_graphs.erase(lru);
        }
        GraphEntry e;
        e.stamp = ++g_gstamp;
        g_graphs.emplace(key, e);
        return false;  // first call: direct
    }
    GraphEntry &e = it->second;
    e.stamp = ++g_gstamp;
    if (!e.exec) {
        cudaStream_t &cs = g_capture_stream[dev];
        cudaError_t err = cudaSuccess;
        if (!cs && (err = cudaStreamCreateWithFlags(&cs, cudaStreamNonBlocking)) != cudaSuccess) {
            cs = nullptr;
            return false;
        }
        // first with conditional nodes (empty passes and lists are skipped on the device),
        // then, if any conditional-graph call fails, as a plain capture
        const uint64_t l0 = g_launches;
        bool done = false;
        for (int attempt = cond_graphs_enabled() ? 0 : 1; attempt < 2 && !done; ++attempt) {
            if (cudaStreamBeginCapture(cs, cudaStreamCaptureModeThreadLocal) != cudaSuccess) return false;
            GraphCtx &gc = g_gctx[dev];
            gc.depth = 0;
            gc.ok = true;
            g_gx = attempt == 0 ? &gc : nullptr;
            g_launches = l0;
            const hrs_status s = run(cs);
            g_gx = nullptr;
            cudaGraph_t g = nullptr;
            err = cudaStreamEndCapture(cs, &g);
            if (s != HRS_SUCCESS || err != cudaSuccess || !g || !gc.ok) {
                if (g) cudaGraphDestroy(g);
                cudaGetLastError();
                continue;
            }
            err = cudaGraphInstantiate(&e.exec, g, 0);
            cudaGraphDestroy(g);
            if (err != cudaSuccess) {
                e.exec = nullptr;
                cudaGetLastError();
                continue;
            }
            done = true;
        }
        if (!done) {
            g_launches = l0;
            return false;  // run directly instead
        }
        e.launches = g_launches - l0;  // (launches captured, including the conditional ones)
        g_launches = l0;               // counted when the graph runs
    }
    const cudaError_t err = cudaGraphLaunch(e.exec, stream);
    if (err != cudaSuccess) {
        *out = cuda_fail(err);
        return true;
    }
    g_launches += e.launches;
    *out = HRS_SUCCESS;
    return true;
}

}  // namespace

// ====================================================================== C ABI

extern "C" {

static hrs_status sort_common(void *d_temp, size_t *temp_bytes, const void *keys_in, void *keys_out,
                              const void *vals_in, void *vals_out, uint64_t n, int key_bytes, int value_bytes,
                              int begin_bit, int end_bit, const hrs_tuning *tuning, const uint64_t *grouped,
                              hrs_stream_t stream, int kind = 0);

hrs_status hrs_sort_ex(void *d_temp, size_t *temp_bytes, const void *keys_in, void *keys_out, const void *vals_in,
                       void *vals_out, uint64_t n, int key_bytes, int value_bytes, int begin_bit, int end_bit,
                       const hrs_tuning *tuning, hrs_stream_t stream) {
    return sort_common(d_temp, temp_bytes, keys_in, keys_out, vals_in, vals_out, n, key_bytes, value_bytes,
                       begin_bit, end_bit, tuning, nullptr, stream);
}

hrs_status hrs_sort_grouped(void *d_temp, size_t *temp_bytes, const void *keys_in, void *keys_out,
                            const void *vals_in, void *vals_out, uint64_t n, int key_bytes, int value_bytes,
                            int begin_bit, int end_bit, const uint64_t *d_first_digit_hist, const hrs_tuning *tuning,
                            hrs_stream_t stream) {
    if (d_temp && n > 0 && begin_bit < end_bit && !d_first_digit_hist) return HRS_ERROR_INVALID_VALUE;
    return sort_common(d_temp, temp_bytes, keys_in, keys_out, vals_in, vals_out, n, key_bytes, value_bytes,
                       begin_bit, end_bit, tuning, d_first_digit_hist, stream);
}

static hrs_status sort_common(void *d_temp, size_t *temp_bytes, const void *keys_in, void *keys_out,
                              const void *vals_in, void *vals_out, uint64_t n, int key_bytes, int value_bytes,
                              int begin_bit, int end_bit, const hrs_tuning *tuning, const uint64_t *grouped,
                              hrs_stream_t stream, int kind) {
    if (!temp_bytes) return HRS_ERROR_INVALID_VALUE;
    if (key_bytes != 4 && key_bytes != 8) return HRS_ERROR_INVALID_VALUE;
    if (value_bytes != 0 && value_bytes != 4 && value_bytes != 8) return HRS_ERROR_INVALID_VALUE;
    if (begin_bit < 0 || end_bit > 8 * key_bytes || begin_bit > end_bit) return HRS_ERROR_INVALID_BITS;
    if (n > HRS_MAX_ITEMS) return HRS_ERROR_TOO_LARGE;
    Plan pl;
    hrs_status s = make_plan(pl, n, key_bytes, value_bytes, begin_bit, end_bit, tuning, MODE_SORT);
    if (s) return s;
    pl.kind = kind;
    if (!d_temp) {
        *temp_bytes = pl.total;
        return HRS_SUCCESS;
    }
    if (*temp_bytes < pl.total) return HRS_ERROR_TEMP_TOO_SMALL;
    if (!aligned(d_temp, 256)) return HRS_ERROR_INVALID_VALUE;
    if (n > 0) {
        if (!keys_in || !keys_out) return HRS_ERROR_INVALID_VALUE;
        if (value_bytes && (!vals_in || !vals_out)) return HRS_ERROR_INVALID_VALUE;
        if (!aligned(keys_in, key_bytes) || !aligned(keys_out, key_bytes)) return HRS_ERROR_INVALID_VALUE;
        if (value_bytes && (!aligned(vals_in, value_bytes) || !aligned(vals_out, value_bytes)))
            return HRS_ERROR_INVALID_VALUE;
        const size_t nk = n * key_bytes, nv = n * value_bytes;
        const void *bufs[5] = {keys_in, keys_out, value_bytes ? vals_in : nullptr, value_bytes ? vals_out : nullptr,
                               d_temp};
        const size_t lens[5] = {nk, nk, nv, nv, pl.total};
        for (int i = 0; i < 5; ++i)
            for (int j = i + 1; j < 5; ++j)
                if (overlap(bufs[i], lens[i], bufs[j], lens[j])) return HRS_ERROR_ALIASING;
    }
    int dev = 0, sms = 0;
    if ((s = check_device(&dev, &sms))) return s;
    cudaStream_t st = reinterpret_cast<cudaStream_t>(stream);
    auto run = [&](cudaStream_t on) {
        return sort_dispatch(key_bytes, value_bytes, pl, d_temp, keys_in, keys_out, vals_in, vals_out, on, dev, sms,
                             grouped);
    };
    cudaStreamCaptureStatus cap = cudaStreamCaptureStatusNone;
    if (n > 0 && n <= HRS_GRAPH_MAX_N && !g_prof && graphs_enabled() &&
        cudaStreamIsCapturing(st, &cap) == cudaSuccess && cap == cudaStreamCaptureStatusNone) {
        GraphKey key;
        std::memset(&key, 0, sizeof(key));
        const hrs_tuning t = tuning ? *tuning : hrs_tuning{};
        uint64_t *v = key.v;
        v[0] = static_cast<uint64_t>(dev);
        v[1] = n;
        v[2] = static_cast<uint64_t>(key_bytes) | (static_cast<uint64_t>(value_bytes) << 8) |
               (static_cast<uint64_t>(begin_bit) << 16) | (static_cast<uint64_t>(end_bit) << 24);
        v[3] = t.local_threshold;
        v[4] = t.merge_threshold;
        v[5] = t.keys_per_tile;
        v[6] = t.local_classes;
        v[7] = reinterpret_cast<uintptr_t>(keys_in);
        v[8] = reinterpret_cast<uintptr_t>(keys_out);
        v[9] = reinterpret_cast<uintptr_t>(vals_in);
        v[10] = reinterpret_cast<uintptr_t>(vals_out);
        v[11] = reinterpret_cast<uintptr_t>(d_temp);
        v[12] = *temp_bytes;
        v[13] = t.flags | env_flags();
        v[14] = reinterpret_cast<uintptr_t>(grouped);
        v[15] = static_cast<uint64_t>(kind);
        hrs_status gs = HRS_SUCCESS;
        if (via_graph(key, st, dev, &gs, run)) return gs;
    }
    return run(st);
}

hrs_status hrs_sort_typed(void *d_temp, size_t *temp_bytes, const void *keys_in, void *keys_out, const void *vals_in,
                          void *vals_out, uint64_t n, int key_bytes, int value_bytes, hrs_key_kind kind,
                          hrs_stream_t stream) {
    if (!temp_bytes) return HRS_ERROR_INVALID_VALUE;
    if (kind != HRS_KEY_UINT && kind != HRS_KEY_INT && kind != HRS_KEY_FLOAT) return HRS_ERROR_INVALID_VALUE;
    if (key_bytes != 4 && key_bytes != 8) return HRS_ERROR_INVALID_VALUE;
    // the bijection is fused into the kernels: a key read from the input is
    // mapped on the way in (histogram, first scatter, local sorts of unmoved buckets) and
    // mapped back where it is written for the last time (last scatter pass, local sorts)
    return sort_common(d_temp, temp_bytes, keys_in, keys_out, vals_in, vals_out, n, key_bytes, value_bytes, 0,
                       8 * key_bytes, nullptr, nullptr, stream, static_cast<int>(kind));
}

}  // extern "C"

namespace {
template <typename K, typename V, int RW, bool KF>
void launch_records(const void *ri, void *ro, void *keys, void *vals, uint64_t n, int kind, int recompose, int grid,
                    cudaStream_t st) {
    LaunchScope ls(st, 4, recompose);
    launch_pdl(k_records<K, V, RW, KF>, dim3(grid), dim3(256), 0, st, static_cast<const uint32_t *>(ri),
               static_cast<uint32_t *>(ro), static_cast<K *>(keys), static_cast<ValT<V> *>(vals), n, kind, recompose);
}
template <typename K, typename V>
void records_kv(bool kf, const void *ri, void *ro, void *keys, void *vals, uint64_t n, int kind, int rc, int grid,
                cudaStream_t st) {
    constexpr int RW = static_cast<int>(sizeof(K) + (HasVal<V>::value ? sizeof(ValT<V>) : 0)) / 4;
    if (kf) launch_records<K, V, RW, true>(ri, ro, keys, vals, n, kind, rc, grid, st);
    else launch_records<K, V, RW, false>(ri, ro, keys, vals, n, kind, rc, grid, st);
}
void records_pass(int kb, int vb, bool kf, const void *ri, void *ro, void *keys, void *vals, uint64_t n, int kind,
                  int rc, int grid, cudaStream_t st) {
    if (kb == 4) {
        if (vb == 0) records_kv<uint32_t, NoVal>(kf, ri, ro, keys, vals, n, kind, rc, grid, st);
        else if (vb == 4) records_kv<uint32_t, uint32_t>(kf, ri, ro, keys, vals, n, kind, rc, grid, st);
        else records_kv<uint32_t, unsigned long long>(kf, ri, ro, keys, vals, n, kind, rc, grid, st);
    } else {
        if (vb == 0) records_kv<unsigned long long, NoVal>(kf, ri, ro, keys, vals, n, kind, rc, grid, st);
        else if (vb == 4) records_kv<unsigned long long, uint32_t>(kf, ri, ro, keys, vals, n, kind, rc, grid, st);
        else records_kv<unsigned long long, unsigned long long>(kf, ri, ro, keys, vals, n, kind, rc, grid, st);
    }
}
}  // namespace

extern "C" {

hrs_status hrs_sort_records(void *d_temp, size_t *temp_bytes, const void *records_in, void *records_out, uint64_t n,
                            int key_bytes, int value_bytes, int key_offset, int begin_bit, int end_bit,
                            hrs_key_kind kind, hrs_stream_t stream) {
    if (!temp_bytes) return HRS_ERROR_INVALID_VALUE;
    if (key_bytes != 4 && key_bytes != 8) return HRS_ERROR_INVALID_VALUE;
    if (value_bytes != 0 && value_bytes != 4 && value_bytes != 8) return HRS_ERROR_INVALID_VALUE;
    if (key_offset != 0 && key_offset != value_bytes) return HRS_ERROR_INVALID_VALUE;
    if (kind != HRS_KEY_UINT && kind != HRS_KEY_INT && kind != HRS_KEY_FLOAT) return HRS_ERROR_INVALID_VALUE;
    if (begin_bit < 0 || end_bit > 8 * key_bytes || begin_bit > end_bit) return HRS_ERROR_INVALID_BITS;
    if (kind != HRS_KEY_UINT && (begin_bit != 0 || end_bit != 8 * key_bytes)) return HRS_ERROR_INVALID_BITS;
    if (n > HRS_MAX_ITEMS) return HRS_ERROR_TOO_LARGE;
    // temp = [keys n*K | values n*V | sorted keys n*K | sorted values n*V | the pair sort's temp]
    size_t inner = 0;
    hrs_status s = hrs_sort_ex(nullptr, &inner, nullptr, nullptr, nullptr, nullptr, n, key_bytes, value_bytes,
                               begin_bit, end_bit, nullptr, stream);
    if (s) return s;
    const size_t nk = align_up(static_cast<size_t>(n) * key_bytes, 256), nv = align_up(static_cast<size_t>(n) * value_bytes, 256);
    const size_t need = 2 * (nk + nv) + inner;
    if (!d_temp) {
        *temp_bytes = need;
        return HRS_SUCCESS;
    }
    if (*temp_bytes < need) return HRS_ERROR_TEMP_TOO_SMALL;
    if (!aligned(d_temp, 256)) return HRS_ERROR_INVALID_VALUE;
    if (n == 0) return HRS_SUCCESS;
    if (!records_in || !records_out || !aligned(records_in, 4) || !aligned(records_out, 4)) return HRS_ERROR_INVALID_VALUE;
    const size_t rb = static_cast<size_t>(n) * (key_bytes + value_bytes);
    if (overlap(records_in, rb, records_out, rb) || overlap(records_in, rb, d_temp, *temp_bytes) ||
        overlap(records_out, rb, d_temp, *temp_bytes))
        return HRS_ERROR_ALIASING;
    int dev = 0, sms = 0;
    if ((s = check_device(&dev, &sms))) return s;
    cudaStream_t st = reinterpret_cast<cudaStream_t>(stream);
    unsigned char *t = static_cast<unsigned char *>(d_temp);
    void *k0 = t, *v0 = t + nk, *k1 = t + nk + nv, *v1 = t + 2 * nk + nv, *inner_t = t + 2 * (nk + nv);
    const int grid = static_cast<int>(std::min<uint64_t>((n + 255) / 256, static_cast<uint64_t>(sms) * 8));
    const bool kf = key_offset == 0;
    records_pass(key_bytes, value_bytes, kf, records_in, nullptr, k0, value_bytes ? v0 : nullptr, n, kind, 0, grid, st);
    if ((s = last_launch())) return s;
    size_t tb = inner;
    if ((s = hrs_sort_ex(inner_t, &tb, k0, k1, value_bytes ? v0 : nullptr, value_bytes ? v1 : nullptr, n, key_bytes,
                         value_bytes, begin_bit, end_bit, nullptr, stream)))
        return s;
    records_pass(key_bytes, value_bytes, kf, nullptr, records_out, k1, value_bytes ? v1 : nullptr, n, kind, 1, grid, st);
    return last_launch();
}

hrs_status hrs_sort_keys_u32(void *t, size_t *tb, const uint32_t *ki, uint32_t *ko, uint64_t n, int b, int e,
                             hrs_stream_t s) {
    return hrs_sort_ex(t, tb, ki, ko, nullptr, nullptr, n, 4, 0, b, e, nullptr, s);
}
hrs_status hrs_sort_keys_u64(void *t, size_t *tb, const uint64_t *ki, uint64_t *ko, uint64_t n, int b, int e,
                             hrs_stream_t s) {
    return hrs_sort_ex(t, tb, ki, ko, nullptr, nullptr, n, 8, 0, b, e, nullptr, s);
}
hrs_status hrs_sort_pairs_u32_u32(void *t, size_t *tb, const uint32_t *ki, uint32_t *ko, const uint32_t *vi,
                                  uint32_t *vo, uint64_t n, int b, int e, hrs_stream_t s) {
    return hrs_sort_ex(t, tb, ki, ko, vi, vo, n, 4, 4, b, e, nullptr, s);
}
hrs_status hrs_sort_pairs_u32_u64(void *t, size_t *tb, const uint32_t *ki, uint32_t *ko, const uint64_t *vi,
                                  uint64_t *vo, uint64_t n, int b, int e, hrs_stream_t s) {
    return hrs_sort_ex(t, tb, ki, ko, vi, vo, n, 4, 8, b, e, nullptr, s);
}
hrs_status hrs_sort_pairs_u64_u32(void *t, size_t *tb, const uint64_t *ki, uint64_t *ko, const uint32_t *vi,
                                  uint32_t *vo, uint64_t n, int b, int e, hrs_stream_t s) {
    return hrs_sort_ex(t, tb, ki, ko, vi, vo, n, 8, 4, b, e, nullptr, s);
}
hrs_status hrs_sort_pairs_u64_u64(void *t, size_t *tb, const uint64_t *ki, uint64_t *ko, const uint64_t *vi,
                                  uint64_t *vo, uint64_t n, int b, int e, hrs_stream_t s) {
    return hrs_sort_ex(t, tb, ki, ko, vi, vo, n, 8, 8, b, e, nullptr, s);
}

hrs_status hrs_get_stats(const void *d_temp, hrs_stats *out, hrs_stream_t stream) {
    if (!d_temp || !out) return HRS_ERROR_INVALID_VALUE;
    Ctl c;
    cudaStream_t st = reinterpret_cast<cudaStream_t>(stream);
    cudaError_t e = cudaMemcpyAsync(&c, d_temp, sizeof(Ctl), cudaMemcpyDeviceToHost, st);
    if (e != cudaSuccess) return cuda_fail(e);
    e = cudaStreamSynchronize(st);
    if (e != cudaSuccess) return cuda_fail(e);
    if (c.magic != CTL_MAGIC) return HRS_ERROR_INVALID_VALUE;
    std::memset(out, 0, sizeof(*out));
    out->n = c.n;
    out->key_bytes = c.key_bytes;
    out->value_bytes = c.value_bytes;
    out->overflow = c.overflow;
    const uint64_t K = c.key_bytes, R = c.key_bytes + c.value_bytes;
    uint64_t bytes = 0;
    for (int p = 1; p <= HRS_MAX_PASSES; ++p) {
        const uint32_t tiles = static_cast<uint32_t>(c.alloc[p] >> 32), bks = static_cast<uint32_t>(c.alloc[p]);
        if (tiles == 0) continue;
        out->counting_passes = p;
        out->recs_in_pass[p - 1] = c.recs_in_pass[p];
        out->tiles_in_pass[p - 1] = tiles;
        out->buckets_in_pass[p - 1] = bks;
        out->skipped_recs_in_pass[p - 1] = c.skipped_in_pass[p];
        // the histogram reads every record of the pass, the scatter moves the unskipped ones
        bytes += c.recs_in_pass[p] * K + (c.recs_in_pass[p] - c.skipped_in_pass[p]) * 2 * R;
    }
    for (int k = 0; k < HRS_NUM_CLASSES; ++k) {
        out->local_in_class[k] = c.nlocal[k];
        out->local_buckets += c.nlocal[k];
    }
    out->local_recs = c.local_recs;
    out->merged_groups = c.merged_groups;
    out->redo_blocks = c.redo;
    out->bytes_min = bytes + c.local_recs * 2 * R;
    return HRS_SUCCESS;
}

uint32_t hrs_max_local_threshold(int key_bytes, int value_bytes) { return max_lt(key_bytes, value_bytes); }
uint32_t hrs_max_keys_per_tile(int key_bytes, int value_bytes) { return max_kpb(key_bytes, value_bytes); }

hrs_status hrs_default_tuning(int key_bytes, int value_bytes, hrs_tuning *out) {
    if (!out || (key_bytes != 4 && key_bytes != 8) || (value_bytes != 0 && value_bytes != 4 && value_bytes != 8))
        return HRS_ERROR_INVALID_VALUE;
    Plan pl;
    hrs_status s = make_plan(pl, 0, key_bytes, value_bytes, 0, 8 * key_bytes, nullptr, MODE_SORT);
    if (s) return s;
    out->local_threshold = pl.lt;
    out->merge_threshold = pl.mt;
    out->keys_per_tile = pl.kpb;
    out->local_classes = 0;
    out->flags = 0;
    return HRS_SUCCESS;
}

uint32_t hrs_class_capacity(int c) { return (c >= 0 && c < HRS_NUM_CLASSES) ? class_capacity(c) : 0u; }

struct DstArgs {
    const uint64_t *offsets;  // host, 2^(hi-lo)
    int nwin;
    const uint64_t *kwin, *vwin;  // host, nwin device addresses
};

static hrs_status block_common(void *d_temp, size_t *temp_bytes, const void *keys_in, void *keys_out,
                               const void *vals_in, void *vals_out, uint64_t n, int kb, int vb, int lo, int hi,
                               uint64_t *h, uint64_t *o, bool scatter, hrs_stream_t stream,
                               const DstArgs *dst = nullptr) {
    if (!temp_bytes) return HRS_ERROR_INVALID_VALUE;
    if (kb != 4 && kb != 8) return HRS_ERROR_INVALID_VALUE;
    if (vb != 0 && vb != 4 && vb != 8) return HRS_ERROR_INVALID_VALUE;
    if (lo < 0 || hi > 8 * kb || hi - lo < 1 || hi - lo > 8) return HRS_ERROR_INVALID_BITS;
    if (n > HRS_MAX_ITEMS) return HRS_ERROR_TOO_LARGE;
    Plan pl;
    hrs_status s = make_plan(pl, n, kb, vb, lo, hi, nullptr, scatter ? MODE_PARTITION : MODE_HIST);
    if (s) return s;
    pl.lo[0] = lo;
    pl.hi[0] = hi;
    if (!d_temp) {
        *temp_bytes = pl.total;
        return HRS_SUCCESS;
    }
    if (*temp_bytes < pl.total) return HRS_ERROR_TEMP_TOO_SMALL;
    if (!aligned(d_temp, 256)) return HRS_ERROR_INVALID_VALUE;
    if (!scatter && !h) return HRS_ERROR_INVALID_VALUE;
    if (n > 0) {
        if (!keys_in || (scatter && !dst && !keys_out)) return HRS_ERROR_INVALID_VALUE;
        if (scatter && !dst && vb && (!vals_in || !vals_out)) return HRS_ERROR_INVALID_VALUE;
        if (!aligned(keys_in, kb) || (scatter && !dst && !aligned(keys_out, kb))) return HRS_ERROR_INVALID_VALUE;
        const size_t nk = n * kb, nv = n * vb;
        const void *bufs[5] = {keys_in, scatter ? keys_out : nullptr, vb ? vals_in : nullptr,
                               vb ? vals_out : nullptr, d_temp};
        const size_t lens[5] = {nk, nk, nv, nv, pl.total};
        for (int i = 0; i < 5; ++i)
            for (int j = i + 1; j < 5; ++j)
                if (overlap(bufs[i], lens[i], bufs[j], lens[j])) return HRS_ERROR_ALIASING;
    }
    int dev = 0, sms = 0;
    if ((s = check_device(&dev, &sms))) return s;
    if (dst) {
        // the window tables into temp (pageable host memory: the copy is staged before the call returns)
        if (!dst->offsets || dst->nwin < 1 || dst->nwin > MAX_WINDOWS || !dst->kwin || (vb && !dst->vwin))
            return HRS_ERROR_INVALID_VALUE;
        const int r = 1 << (hi - lo);
        std::vector<uint64_t> tab(RADIX + 2 * MAX_WINDOWS, 0);
        for (int d = 0; d < r; ++d) {
            if ((dst->offsets[d] >> 48) >= static_cast<uint64_t>(dst->nwin)) return HRS_ERROR_INVALID_VALUE;
            tab[d] = dst->offsets[d];
        }
        for (int w = 0; w < dst->nwin; ++w) {
            if (!dst->kwin[w] || (dst->kwin[w] % kb) || (vb && (!dst->vwin[w] || dst->vwin[w] % vb)))
                return HRS_ERROR_INVALID_VALUE;
            tab[RADIX + w] = dst->kwin[w];
            tab[RADIX + MAX_WINDOWS + w] = vb ? dst->vwin[w] : 0;
        }
        cudaStream_t st = reinterpret_cast<cudaStream_t>(stream);
        cudaError_t e = cudaMemcpyAsync(static_cast<unsigned char *>(d_temp) + pl.off_dst, tab.data(),
                                        sizeof(uint64_t) * tab.size(), cudaMemcpyHostToDevice, st);
        if (e != cudaSuccess) return cuda_fail(e);
        e = cudaStreamSynchronize(st);  // (tab is a local: the copy must be done before it goes)
        if (e != cudaSuccess) return cuda_fail(e);
        pl.dst = true;
    }
    return block_dispatch(kb, vb, pl, d_temp, keys_in, keys_out, vals_in, vals_out, h, o, scatter,
                          reinterpret_cast<cudaStream_t>(stream), dev, sms);
}

hrs_status hrs_digit_histogram(void *d_temp, size_t *temp_bytes, const void *keys, uint64_t n, int key_bytes,
                               int lo_bit, int hi_bit, uint64_t *d_hist, hrs_stream_t stream) {
    return block_common(d_temp, temp_bytes, keys, nullptr, nullptr, nullptr, n, key_bytes, 0, lo_bit, hi_bit,
                        d_hist, nullptr, false, stream);
}

hrs_status hrs_partition_pass_to(void *d_temp, size_t *temp_bytes, const void *keys_in, const void *vals_in,
                                 uint64_t n, int key_bytes, int value_bytes, int lo_bit, int hi_bit,
                                 const uint64_t *dst_offsets, int nwindows, const uint64_t *key_windows,
                                 const uint64_t *value_windows, hrs_stream_t stream) {
    DstArgs da{dst_offsets, nwindows, key_windows, value_windows};
    return block_common(d_temp, temp_bytes, keys_in, nullptr, vals_in, nullptr, n, key_bytes, value_bytes, lo_bit,
                        hi_bit, nullptr, nullptr, true, stream, d_temp ? &da : nullptr);
}

hrs_status hrs_partition_pass(void *d_temp, size_t *temp_bytes, const void *keys_in, void *keys_out,
                              const void *vals_in, void *vals_out, uint64_t n, int key_bytes, int value_bytes,
                              int lo_bit, int hi_bit, uint64_t *d_offsets, hrs_stream_t stream) {
    return block_common(d_temp, temp_bytes, keys_in, keys_out, vals_in, vals_out, n, key_bytes, value_bytes, lo_bit,
                        hi_bit, nullptr, d_offsets, true, stream);
}

hrs_status hrs_copy_pieces(void *dst, const void *src, int elem_bytes, const uint64_t *pieces, uint64_t npieces,
                           hrs_stream_t stream) {
    if (elem_bytes != 4 && elem_bytes != 8) return HRS_ERROR_INVALID_VALUE;
    if (npieces == 0) return HRS_SUCCESS;
    if (!dst || !src || !pieces) return HRS_ERROR_INVALID_VALUE;
    if (!aligned(dst, elem_bytes) || !aligned(src, elem_bytes)) return HRS_ERROR_INVALID_VALUE;
    int dev = 0, sms = 0;
    hrs_status s = check_device(&dev, &sms);
    if (s) return s;
    cudaStream_t st = reinterpret_cast<cudaStream_t>(stream);
    for (uint64_t p0 = 0; p0 < npieces; p0 += COPY_PIECES_MAX) {  // the table goes in the kernel parameters
        CopyPieces cp;
        cp.npieces = static_cast<uint32_t>(std::min<uint64_t>(COPY_PIECES_MAX, npieces - p0));
        std::memcpy(cp.tab, pieces + 3 * p0, sizeof(uint64_t) * 3 * cp.npieces);
        LaunchScope ls(st, 4, 0);
        if (elem_bytes == 4)
            launch_pdl(k_copy_pieces<uint32_t>, dim3(sms * 4), dim3(256), 0, st, static_cast<const uint32_t *>(src),
                       static_cast<uint32_t *>(dst), cp);
        else
            launch_pdl(k_copy_pieces<unsigned long long>, dim3(sms * 4), dim3(256), 0, st,
                       static_cast<const unsigned long long *>(src), static_cast<unsigned long long *>(dst), cp);
        if ((s = last_launch())) return s;
    }
    return HRS_SUCCESS;
}

const char *hrs_status_string(hrs_status s) {
    switch (s) {
        case HRS_SUCCESS: return "success";
        case HRS_ERROR_INVALID_VALUE: return "invalid value";
        case HRS_ERROR_INVALID_BITS: return "invalid bit range";
        case HRS_ERROR_ALIASING: return "buffers overlap";
        case HRS_ERROR_TEMP_TOO_SMALL: return "temp storage too small";
        case HRS_ERROR_TOO_LARGE: return "n exceeds HRS_MAX_ITEMS";
        case HRS_ERROR_NO_DEVICE: return "current device is not an sm_100 GPU";
        case HRS_ERROR_CUDA: return "CUDA error";
    }
    return "unknown status";
}

int hrs_last_cuda_error(void) { return g_last_cuda; }
uint64_t hrs_launch_count(void) { return g_launches; }

void hrs_profile_enable(int on) {
    for (auto &r : g_prof_recs) {
        g_prof_pool.push_back(r.a);
        g_prof_pool.push_back(r.b);
    }
    g_prof_recs.clear();
    g_prof = on != 0;
}

int hrs_profile_collect(hrs_profile_record *out, int max) {
    int k = 0;
    for (auto &r : g_prof_recs) {
        if (out && k < max) {
            float ms = 0.f;
            cudaEventSynchronize(r.b);
            cudaEventElapsedTime(&ms, r.a, r.b);
            out[k].kind = r.kind;
            out[k].pass = r.pass;
            out[k].ms = ms;
            ++k;
        }
        g_prof_pool.push_back(r.a);
        g_prof_pool.push_back(r.b);
    }
    g_prof_recs.clear();
    return k;
}
int hrs_version(void) { return 1; }

}  // extern "C"
