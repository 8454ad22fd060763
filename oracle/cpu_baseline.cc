/*
 * cpu_baseline.cc -- CPU reference programs for the hybrid radix sort benchmark
 * (arXiv 1611.01137; /root/reference/PAPER.md cited as P:<line>).
 *
 * TEST INFRASTRUCTURE ONLY, like oracle.c: only tests/, __graft_entry__.smoke() and
 * bench.py's cpu_baseline / --impl reference legs may load or call this code.  It
 * shares no code, header, table or constant with the CUDA library, and the library
 * never calls it (there is no CPU fallback).
 *
 * Two programs, both computing THE result of the method -- the unique stable sort of
 * the records by key bits [begin, end):
 *
 *   cpu_lsd_sort     the timed CPU baseline of SURVEY.md §8(d): the LSD radix sort of
 *                    P:304-311 with 8-bit digits, each pass a stable
 *                    counting sort (histogram, exclusive prefix sum, scatter in input
 *                    order, P:293-301 / P:503-509) split over T host threads.  Thread t
 *                    owns the contiguous chunk [t*n/T, (t+1)*n/T); its digit-d records
 *                    are placed after those of every digit < d and after the digit-d
 *                    records of threads < t, i.e. exactly where the one-thread pass puts
 *                    them: the output is byte-identical to oracle_lsd_sort for any T.
 *                    Native key / value widths (4 or 8 bytes; values optional).
 *   cpu_stable_sort  std::stable_sort of (key, value) records with the comparator
 *                    sk(a) < sk(b), one thread: the library routine the oracle is
 *                    cross-checked against (BJ north_star), and a second timed baseline.
 *
 * Return 0 on success, 1 on invalid arguments, 2 when allocation fails.
 */
#include <algorithm>
#include <cstdint>
#include <cstring>
#include <new>
#include <thread>
#include <vector>

namespace {

template <typename K>
inline uint32_t digit(K key, int lo, int width) {
    return static_cast<uint32_t>((static_cast<uint64_t>(key) >> lo) & ((uint64_t(1) << width) - 1));
}

template <typename K, typename V>
int lsd(const K *keys, const V *vals, uint64_t n, int begin, int end, K *keys_out, V *vals_out, int threads) {
    if (begin < 0 || end > int(8 * sizeof(K)) || begin > end || threads < 1) return 1;
    if (n == 0) return 0;
    std::memcpy(keys_out, keys, sizeof(K) * n);
    if (vals) std::memcpy(vals_out, vals, sizeof(V) * n);
    if (begin == end) return 0;
    K *k2 = new (std::nothrow) K[n];
    V *v2 = vals ? new (std::nothrow) V[n] : nullptr;
    if (!k2 || (vals && !v2)) {
        delete[] k2;
        delete[] v2;
        return 2;
    }
    const int T = static_cast<int>(std::min<uint64_t>(threads, n));
    std::vector<uint64_t> cnt(static_cast<size_t>(T) * 256);
    K *ks = keys_out, *kd = k2;
    V *vs = vals_out, *vd = v2;
    int npass = 0;
    auto run = [&](auto &&fn) {
        std::vector<std::thread> th;
        for (int t = 1; t < T; ++t) th.emplace_back(fn, t);
        fn(0);
        for (auto &x : th) x.join();
    };
    for (int lo = begin; lo < end; lo += 8) {
        const int width = std::min(8, end - lo);
        const uint32_t radix = 1u << width;
        // (1) per-thread histograms of the thread's chunk
        run([&](int t) {
            uint64_t *c = &cnt[static_cast<size_t>(t) * 256];
            std::fill(c, c + 256, 0);
            const uint64_t a = n * t / T, b = n * (t + 1) / T;
            for (uint64_t i = a; i < b; ++i) ++c[digit(ks[i], lo, width)];
        });
        // (2) exclusive prefix over (digit, thread) in that order
        uint64_t run_sum = 0;
        for (uint32_t d = 0; d < radix; ++d)
            for (int t = 0; t < T; ++t) {
                uint64_t &c = cnt[static_cast<size_t>(t) * 256 + d];
                const uint64_t x = c;
                c = run_sum;
                run_sum += x;
            }
        // (3) every thread scatters its chunk in input order
        run([&](int t) {
            uint64_t *pos = &cnt[static_cast<size_t>(t) * 256];
            const uint64_t a = n * t / T, b = n * (t + 1) / T;
            for (uint64_t i = a; i < b; ++i) {
                const uint32_t d = digit(ks[i], lo, width);
                const uint64_t p = pos[d]++;
                kd[p] = ks[i];
                if (vals) vd[p] = vs[i];
            }
        });
        std::swap(ks, kd);
        std::swap(vs, vd);
        ++npass;
    }
    if (npass & 1) {  // the result is in the scratch buffers
        std::memcpy(keys_out, ks, sizeof(K) * n);
        if (vals) std::memcpy(vals_out, vs, sizeof(V) * n);
    }
    delete[] k2;
    delete[] v2;
    return 0;
}

template <typename K, typename V>
int stable(const K *keys, const V *vals, uint64_t n, int begin, int end, K *keys_out, V *vals_out) {
    if (begin < 0 || end > int(8 * sizeof(K)) || begin > end) return 1;
    const int w = end - begin;
    const uint64_t mask = w >= 64 ? ~uint64_t(0) : ((uint64_t(1) << w) - 1);
    auto sk = [&](K x) { return w == 0 ? uint64_t(0) : ((static_cast<uint64_t>(x) >> begin) & mask); };
    struct Rec {
        K k;
        V v;
    };
    std::vector<Rec> r;
    try {
        r.resize(n);
    } catch (...) {
        return 2;
    }
    for (uint64_t i = 0; i < n; ++i) r[i] = Rec{keys[i], vals ? vals[i] : V(0)};
    std::stable_sort(r.begin(), r.end(), [&](const Rec &a, const Rec &b) { return sk(a.k) < sk(b.k); });
    for (uint64_t i = 0; i < n; ++i) {
        keys_out[i] = r[i].k;
        if (vals) vals_out[i] = r[i].v;
    }
    return 0;
}

}  // namespace

extern "C" {

int cpu_lsd_sort(const void *keys, const void *vals, uint64_t n, int key_bytes, int value_bytes, int begin,
                 int end, void *keys_out, void *vals_out, int threads) {
#define HRS_CPU_LSD(K, V)                                                                                     \
    return lsd<K, V>(static_cast<const K *>(keys), static_cast<const V *>(value_bytes ? vals : nullptr), n,  \
                     begin, end, static_cast<K *>(keys_out), static_cast<V *>(value_bytes ? vals_out : nullptr), \
                     threads)
    if (key_bytes == 4 && (value_bytes == 0 || value_bytes == 4)) HRS_CPU_LSD(uint32_t, uint32_t);
    if (key_bytes == 4 && value_bytes == 8) HRS_CPU_LSD(uint32_t, uint64_t);
    if (key_bytes == 8 && (value_bytes == 0 || value_bytes == 4)) HRS_CPU_LSD(uint64_t, uint32_t);
    if (key_bytes == 8 && value_bytes == 8) HRS_CPU_LSD(uint64_t, uint64_t);
#undef HRS_CPU_LSD
    return 1;
}

int cpu_stable_sort(const void *keys, const void *vals, uint64_t n, int key_bytes, int value_bytes, int begin,
                    int end, void *keys_out, void *vals_out) {
#define HRS_CPU_STABLE(K, V)                                                                                     \
    return stable<K, V>(static_cast<const K *>(keys), static_cast<const V *>(value_bytes ? vals : nullptr), n,  \
                        begin, end, static_cast<K *>(keys_out), static_cast<V *>(value_bytes ? vals_out : nullptr))
    if (key_bytes == 4 && (value_bytes == 0 || value_bytes == 4)) HRS_CPU_STABLE(uint32_t, uint32_t);
    if (key_bytes == 4 && value_bytes == 8) HRS_CPU_STABLE(uint32_t, uint64_t);
    if (key_bytes == 8 && (value_bytes == 0 || value_bytes == 4)) HRS_CPU_STABLE(uint64_t, uint32_t);
    if (key_bytes == 8 && value_bytes == 8) HRS_CPU_STABLE(uint64_t, uint64_t);
#undef HRS_CPU_STABLE
    return 1;
}

}  // extern "C"
