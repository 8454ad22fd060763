// hrs_device.cuh -- sm_100a kernels of the stable hybrid MSD radix sort.
//
// Paper: Stehle & Jacobsen, arXiv 1611.01137 (PAPER.md lines cited as P:<line>).
// Every pass p of the MSD recursion (Fig 1) runs two kernels over a
// device-resident tile table ("key blocks"), so each pass costs a
// constant number of launches and the host never reads device memory:
//
//   k_hist<p>     per tile: digit histogram with warp-aggregated shared-memory
//                 atomics (Fig 2), then a decoupled look-back across the
//                 tiles of the same bucket that turns tile histograms into
//                 tile-ordered prefix sums (replaces the atomicAdd chunk
//                 reservation of P:696-703, which is not stable).  The last tile of
//                 every bucket owns the bucket's histogram: it computes the
//                 sub-bucket offsets (exclusive prefix sum) and classifies
//                 the sub-buckets (R1-R3 P:805-811, merging P:552-561), writing the
//                 next pass's tile/bucket tables and the local-sort lists.
//   k_scatter<p>  per tile: stable in-tile rank (warp match-any multisplit with
//                 per-warp digit counters), staging in shared memory, and
//                 coalesced write-combined stores of every digit run to its
//                 sub-bucket (Fig 3); values follow their keys.
//
// then one k_local launch per size class sorts every bucket of at most
// ∂ˆ records on chip with a stable LSD radix sort over the remaining bits
// (P:474-480), skipping digits that are constant across the bucket.
//
// Stability everywhere (ties keep input order) is the one deliberate departure
// from the paper: the output is the unique stable sort.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

#include <type_traits>

#include "../../include/hrs.h"

namespace hrs {

constexpr int RADIX = 256;
constexpr int NBINS = 257;            // 256 digit values + 1 bin for padding lanes
constexpr uint32_t INVALID_DIGIT = 256;
constexpr uint64_t CTL_MAGIC = 0x4852535f31363131ull;  // "HRS_1611"

enum SrcCode : uint16_t { SRC_IN = 0, SRC_AUX = 1, SRC_OUT = 2 };

// One tile ("key block"): up to KPB consecutive records of one bucket.
struct Tile {
    uint64_t offs;
    uint32_t count;
    uint32_t bucket;
};
// A bucket that is counting-sorted in the current pass; its tiles are
// first_tile .. first_tile + ntiles - 1, consecutive and in memory order (the
// order the look-back follows, which makes the pass stable).
struct Bucket {
    uint64_t offs;
    uint32_t count;
    uint32_t first_tile;
    uint32_t ntiles;
    uint32_t pad;
};
// A local-sort assignment: bits [begin_bit, hi_bit) remain to sort.
struct LocalEntry {
    uint64_t offs;
    uint32_t count;
    uint16_t hi_bit;
    uint16_t src;
};

// Control / statistics block at offset 0 of temp.  Zeroed by k_init on every call.
struct Ctl {
    unsigned long long magic;
    unsigned long long n;
    uint32_t key_bytes, value_bytes;
    uint32_t ntiles[HRS_MAX_PASSES + 2];    // tiles of pass p (1-based)
    uint32_t nbuckets[HRS_MAX_PASSES + 2];  // buckets of pass p
    uint32_t claim[HRS_MAX_PASSES + 2];     // dynamic tile claims of k_hist, pass p
    uint32_t nlocal[HRS_NUM_CLASSES];       // entries in local list c
    uint32_t overflow;
    uint32_t pad_;
    unsigned long long recs_in_pass[HRS_MAX_PASSES + 2];
    unsigned long long local_recs;
    unsigned long long merged_groups;
};

// ------------------------------------------------------------------ small helpers

__device__ __forceinline__ uint32_t lanemask_lt() {
    uint32_t r;
    asm("mov.u32 %0, %%lanemask_lt;" : "=r"(r));
    return r;
}

template <typename K>
__device__ __forceinline__ uint32_t digit_of(K key, int lo, uint32_t mask) {
    return static_cast<uint32_t>(key >> lo) & mask;
}

template <typename S>
struct StatusBits;
template <>
struct StatusBits<uint32_t> {
    static constexpr uint32_t AGG = 1u << 30, INC = 2u << 30, FLAGS = 3u << 30, VAL = (1u << 30) - 1;
};
template <>
struct StatusBits<unsigned long long> {
    static constexpr unsigned long long AGG = 1ull << 62, INC = 2ull << 62, FLAGS = 3ull << 62,
                                        VAL = (1ull << 62) - 1;
};

template <typename T>
__device__ __forceinline__ T ld_volatile(const T *p) {
    return *reinterpret_cast<const volatile T *>(p);
}
template <typename T>
__device__ __forceinline__ void st_volatile(T *p, T v) {
    *reinterpret_cast<volatile T *>(p) = v;
}

struct NoVal {};
template <typename V>
struct HasVal {
    static constexpr bool value = true;
};
template <>
struct HasVal<NoVal> {
    static constexpr bool value = false;
};

__host__ __device__ __forceinline__ int size_class_of(uint32_t size) {
    int c = 0;
    while ((128u << c) < size && c < HRS_NUM_CLASSES - 1) ++c;
    return c;
}

// Exclusive scan of n <= 288 u32 values in shared memory, in place, by warp 0.
// Returns nothing; caller syncs before and after.
__device__ __forceinline__ void warp0_exclusive_scan(uint32_t *a, int n) {
    if (threadIdx.x >= 32) return;
    const int lane = threadIdx.x;
    constexpr int PER = 9;  // 32 * 9 = 288 >= 257
    uint32_t v[PER];
    uint32_t s = 0;
#pragma unroll
    for (int i = 0; i < PER; ++i) {
        int idx = lane * PER + i;
        v[i] = idx < n ? a[idx] : 0u;
        s += v[i];
    }
    uint32_t incl = s;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
        uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
        if (lane >= o) incl += y;
    }
    uint32_t run = incl - s;
#pragma unroll
    for (int i = 0; i < PER; ++i) {
        int idx = lane * PER + i;
        if (idx < n) a[idx] = run;
        run += v[i];
    }
}

// ------------------------------------------------------------------ init / copy

struct InitParams {
    Ctl *ctl;
    Tile *tiles;       // pass-1 tile table
    Bucket *buckets;   // pass-1 bucket table
    void *status;      // pass-1 status array (to clear)
    int status_bytes;  // sizeof(S)
    LocalEntry *root_local;  // list of the root's size class (n <= ∂ˆ)
    int root_class;
    uint64_t n;
    uint32_t kpb;
    int counting;      // 1: the root bucket is counting-sorted
    int end_bit;
    uint32_t key_bytes, value_bytes;
};

__global__ void k_init(InitParams prm) {
    const uint64_t n = prm.n;
    const uint32_t T1 = prm.counting ? static_cast<uint32_t>((n + prm.kpb - 1) / prm.kpb) : 0u;
    if (blockIdx.x == 0) {
        uint32_t *w = reinterpret_cast<uint32_t *>(prm.ctl);
        for (int i = threadIdx.x; i < static_cast<int>(sizeof(Ctl) / 4); i += blockDim.x) w[i] = 0;
        __syncthreads();
        if (threadIdx.x == 0) {
            Ctl *c = prm.ctl;
            c->magic = CTL_MAGIC;
            c->n = n;
            c->key_bytes = prm.key_bytes;
            c->value_bytes = prm.value_bytes;
            if (prm.counting) {
                c->ntiles[1] = T1;
                c->nbuckets[1] = 1;
                c->recs_in_pass[1] = n;
                Bucket b;
                b.offs = 0;
                b.count = static_cast<uint32_t>(n);
                b.first_tile = 0;
                b.ntiles = T1;
                b.pad = 0;
                prm.buckets[0] = b;
            } else if (n > 0 && prm.root_local) {
                LocalEntry e;
                e.offs = 0;
                e.count = static_cast<uint32_t>(n);
                e.hi_bit = static_cast<uint16_t>(prm.end_bit);
                e.src = SRC_IN;
                prm.root_local[0] = e;
                c->nlocal[prm.root_class] = 1;
                c->local_recs = n;
            }
        }
    }
    const uint64_t stride = static_cast<uint64_t>(gridDim.x) * blockDim.x;
    const uint64_t tid = static_cast<uint64_t>(blockIdx.x) * blockDim.x + threadIdx.x;
    for (uint64_t t = tid; t < T1; t += stride) {
        Tile tl;
        tl.offs = t * prm.kpb;
        tl.count = static_cast<uint32_t>(min(static_cast<uint64_t>(prm.kpb), n - tl.offs));
        tl.bucket = 0;
        prm.tiles[t] = tl;
    }
    // clear the pass-1 look-back status words (16-byte stores)
    const uint64_t words16 = (static_cast<uint64_t>(T1) * RADIX * prm.status_bytes) / 16;
    uint4 *s = reinterpret_cast<uint4 *>(prm.status);
    for (uint64_t i = tid; i < words16; i += stride) s[i] = make_uint4(0, 0, 0, 0);
}

template <typename T>
__global__ void k_copy(const T *__restrict__ in, T *__restrict__ out, uint64_t n) {
    const uint64_t stride = static_cast<uint64_t>(gridDim.x) * blockDim.x;
    for (uint64_t i = static_cast<uint64_t>(blockIdx.x) * blockDim.x + threadIdx.x; i < n; i += stride)
        out[i] = in[i];
}

__global__ void k_fill_u64(uint64_t *p, uint64_t n, uint64_t v) {
    for (uint64_t i = static_cast<uint64_t>(blockIdx.x) * blockDim.x + threadIdx.x; i < n;
         i += static_cast<uint64_t>(gridDim.x) * blockDim.x)
        p[i] = v;
}

// ------------------------------------------------------------------ histogram + look-back + classify

struct HistParams {
    const void *keys;  // X_{p-1}
    int p;
    int last;          // 1: digit p is the least-significant one (no further classification)
    int lo;            // digit bits [lo, lo + width)
    int width;
    uint32_t mask;
    const Tile *tiles;
    const Bucket *buckets;
    Tile *next_tiles;
    Bucket *next_buckets;
    void *status;
    uint32_t *sub_rel;  // [bucket][256] sub-bucket starts relative to the bucket
    Ctl *ctl;
    LocalEntry *local[HRS_NUM_CLASSES];
    uint32_t local_cap[HRS_NUM_CLASSES];
    uint32_t tile_cap, bucket_cap;
    uint32_t lt, mt, kpb;
    int single_class;  // >= 0: every local entry goes to this class (ablation)
    uint16_t src_code; // buffer holding X_p
    uint64_t *out_hist;     // building block: the root bucket's histogram
    uint64_t *out_offsets;  // building block: the root bucket's sub-bucket starts (+ n)
};

template <typename K>
__device__ __forceinline__ void hist_add(uint32_t *hist, uint32_t d) {
    // warp-aggregated shared-memory atomic: one atomicAdd per group of equal digits
    const uint32_t m = __match_any_sync(0xffffffffu, d);
    if (d != INVALID_DIGIT && (m & lanemask_lt()) == 0) atomicAdd(&hist[d], static_cast<uint32_t>(__popc(m)));
}

template <typename K, typename S, int THREADS>
__device__ void classify_bucket(const HistParams &prm, const Bucket &bk, uint32_t bucket_id, const S *tot_in,
                                uint32_t *sm) {
    // sm: scratch of >= 8 * 257 u32
    uint32_t *tot = sm;                 // 256 (+1)
    uint32_t *start = sm + 1 * NBINS;   // exclusive prefix of tot
    uint32_t *ct = sm + 2 * NBINS;      // child tiles per digit -> exclusive
    uint32_t *cb = sm + 3 * NBINS;      // child flag per digit -> exclusive
    uint32_t *glead = sm + 4 * NBINS;   // local group size at the leader digit (0 = none)
    uint32_t *gmulti = sm + 5 * NBINS;  // 1 if the group merged >= 2 sub-buckets
    uint32_t *misc = sm + 6 * NBINS;    // [0] base tile, [1] base bucket, [2..9] class counts, [10..17] class bases
    const int tid = threadIdx.x;
    const S VAL = StatusBits<S>::VAL;
    for (int d = tid; d < NBINS; d += THREADS) {
        uint32_t v = d < RADIX ? static_cast<uint32_t>(tot_in[d] & VAL) : 0u;
        tot[d] = v;
        start[d] = v;
        glead[d] = 0;
        gmulti[d] = 0;
        bool cnt = !prm.last && v > prm.lt;
        ct[d] = cnt ? (v + prm.kpb - 1) / prm.kpb : 0u;
        cb[d] = cnt ? 1u : 0u;
    }
    if (tid < 32) misc[tid] = 0;
    __syncthreads();
    // three exclusive scans, one per warp
    if (tid < 32) warp0_exclusive_scan(start, NBINS);
    __syncthreads();
    if (tid < 32) warp0_exclusive_scan(ct, NBINS);
    __syncthreads();
    if (tid < 32) warp0_exclusive_scan(cb, NBINS);
    __syncthreads();
    const uint64_t boffs = bk.offs;
    for (int d = tid; d < RADIX; d += THREADS) prm.sub_rel[static_cast<uint64_t>(bucket_id) * RADIX + d] = start[d];
    if (prm.out_hist)
        for (int d = tid; d < (1 << prm.width); d += THREADS) prm.out_hist[d] = tot[d];
    if (prm.out_offsets) {
        for (int d = tid; d < (1 << prm.width); d += THREADS) prm.out_offsets[d] = boffs + start[d];
        if (tid == 0) prm.out_offsets[1 << prm.width] = boffs + bk.count;
    }
    if (prm.last) return;

    // ---- counting children: next-pass buckets and their tiles (R2, R4)
    const uint32_t TT = ct[RADIX];  // exclusive scan over 257 entries: ct[256] = total
    const uint32_t NC = cb[RADIX];
    if (tid == 0) {
        uint32_t bt = 0, bb = 0;
        if (NC) {
            bt = atomicAdd(&prm.ctl->ntiles[prm.p + 1], TT);
            bb = atomicAdd(&prm.ctl->nbuckets[prm.p + 1], NC);
            if (bt + TT > prm.tile_cap || bb + NC > prm.bucket_cap) atomicExch(&prm.ctl->overflow, 1u);
        }
        misc[0] = bt;
        misc[1] = bb;
    }
    // ---- local candidates: greedy merge (R3 / reading #5)
    bool has_small = false;
    for (int d = tid; d < RADIX; d += THREADS) {
        uint32_t s = tot[d];
        if (s > 0 && s <= prm.lt && s < prm.mt) has_small = true;
    }
    has_small = __syncthreads_or(has_small);
    if (!has_small) {
        // no sub-bucket can merge: every candidate is its own group
        for (int d = tid; d < RADIX; d += THREADS) {
            uint32_t s = tot[d];
            if (s > 0 && s <= prm.lt) glead[d] = s;
        }
    } else if (tid == 0) {
        int gl = -1;
        uint32_t gs = 0, gc = 0;
        for (int d = 0; d < RADIX; ++d) {
            uint32_t s = tot[d];
            if (s == 0) continue;
            if (s > prm.lt) {
                if (gl >= 0) { glead[gl] = gs; gmulti[gl] = gc > 1; }
                gl = -1;
                continue;
            }
            if (gl >= 0 && gs + s < prm.mt) {
                gs += s;
                ++gc;
            } else {
                if (gl >= 0) { glead[gl] = gs; gmulti[gl] = gc > 1; }
                gl = d;
                gs = s;
                gc = 1;
            }
        }
        if (gl >= 0) { glead[gl] = gs; gmulti[gl] = gc > 1; }
    }
    __syncthreads();
    // per-class slot allocation
    uint32_t my_slot[(RADIX + THREADS - 1) / THREADS];
    int my_cls[(RADIX + THREADS - 1) / THREADS];
#pragma unroll
    for (int i = 0; i < (RADIX + THREADS - 1) / THREADS; ++i) {
        int d = tid + i * THREADS;
        my_cls[i] = -1;
        if (d < RADIX && glead[d]) {
            int c = prm.single_class >= 0 ? prm.single_class : size_class_of(glead[d]);
            my_cls[i] = c;
            my_slot[i] = atomicAdd(&misc[2 + c], 1u);
        }
    }
    __syncthreads();
    if (tid < HRS_NUM_CLASSES) {
        uint32_t cnt = misc[2 + tid];
        uint32_t base = cnt ? atomicAdd(&prm.ctl->nlocal[tid], cnt) : 0u;
        if (base + cnt > prm.local_cap[tid]) atomicExch(&prm.ctl->overflow, 1u);
        misc[10 + tid] = base;
    }
    if (tid == 32) {
        // statistics: records of the next pass, local records, merged groups
        unsigned long long recs_next = 0, lrecs = 0, merged = 0;
        for (int d = 0; d < RADIX; ++d) {
            uint32_t s = tot[d];
            if (!prm.last && s > prm.lt) recs_next += s;
            if (glead[d]) { lrecs += glead[d]; merged += gmulti[d]; }
        }
        if (recs_next) atomicAdd(&prm.ctl->recs_in_pass[prm.p + 1], recs_next);
        if (lrecs) atomicAdd(&prm.ctl->local_recs, lrecs);
        if (merged) atomicAdd(&prm.ctl->merged_groups, merged);
    }
    __syncthreads();
    const int hi_p = prm.lo + prm.width;
#pragma unroll
    for (int i = 0; i < (RADIX + THREADS - 1) / THREADS; ++i) {
        int d = tid + i * THREADS;
        if (my_cls[i] >= 0) {
            int c = my_cls[i];
            uint32_t slot = misc[10 + c] + my_slot[i];
            if (slot < prm.local_cap[c]) {
                LocalEntry e;
                e.offs = boffs + start[d];
                e.count = glead[d];
                e.hi_bit = static_cast<uint16_t>(gmulti[d] ? hi_p : prm.lo);
                e.src = prm.src_code;
                prm.local[c][slot] = e;
            }
        }
    }
    // child buckets
    const uint32_t bt = misc[0], bb = misc[1];
    for (int d = tid; d < RADIX; d += THREADS) {
        uint32_t s = tot[d];
        if (!(s > prm.lt)) continue;
        uint32_t id = bb + cb[d];
        if (id >= prm.bucket_cap) continue;
        Bucket nb;
        nb.offs = boffs + start[d];
        nb.count = s;
        nb.first_tile = bt + ct[d];
        nb.ntiles = (s + prm.kpb - 1) / prm.kpb;
        nb.pad = 0;
        prm.next_buckets[id] = nb;
    }
    // child tiles, spread over the block (a child can own many tiles)
    for (uint32_t i = tid; i < TT; i += THREADS) {
        // find digit d with ct[d] <= i < ct[d+1]
        int lo = 0, hi = RADIX - 1;
        while (lo < hi) {
            int mid = (lo + hi + 1) >> 1;
            if (ct[mid] <= i) lo = mid; else hi = mid - 1;
        }
        // skip digits with zero child tiles sharing the same start
        int d = lo;
        while (d < RADIX - 1 && ct[d + 1] <= i) ++d;
        const uint32_t k = i - ct[d];
        const uint32_t s = tot[d];
        if (bt + i >= prm.tile_cap) continue;
        Tile tl;
        tl.offs = boffs + start[d] + static_cast<uint64_t>(k) * prm.kpb;
        tl.count = min(prm.kpb, s - k * prm.kpb);
        tl.bucket = bb + cb[d];
        prm.next_tiles[bt + i] = tl;
    }
}

template <typename K, typename S, int THREADS>
__global__ void __launch_bounds__(THREADS) k_hist(HistParams prm) {
    static_assert(THREADS >= RADIX, "one thread per digit in the look-back");
    __shared__ uint32_t hist[RADIX];
    __shared__ uint32_t s_tile;
    __shared__ S tot[RADIX];
    __shared__ uint32_t scratch[8 * NBINS];
    using SB = StatusBits<S>;
    const K *__restrict__ keys = static_cast<const K *>(prm.keys);
    S *status = static_cast<S *>(prm.status);
    Ctl *ctl = prm.ctl;
    const uint32_t T = ctl->ntiles[prm.p];
    const int tid = threadIdx.x;
    constexpr int VK = 16 / sizeof(K);  // keys per 16-byte vector
    constexpr int U = 4;                // vectors in flight per thread

    for (;;) {
        if (tid == 0) s_tile = atomicAdd(&ctl->claim[prm.p], 1u);
        for (int i = tid; i < RADIX; i += THREADS) hist[i] = 0;
        __syncthreads();
        const uint32_t t = s_tile;
        if (t >= T) break;
        const Tile tile = prm.tiles[t];
        const K *src = keys + tile.offs;
        const uint32_t count = tile.count;
        // ---- histogram: scalar head up to 16-byte alignment, 16-byte vectors, scalar tail
        const uint32_t mis = static_cast<uint32_t>((reinterpret_cast<uintptr_t>(src) & 15u) / sizeof(K));
        const uint32_t head = min(count, mis ? static_cast<uint32_t>(VK) - mis : 0u);
        const uint32_t nvec = (count - head) / VK;
        const uint32_t tail0 = head + nvec * VK;
        if (tid < 32) {
            const uint32_t ntail = count - tail0;
            const uint32_t u = static_cast<uint32_t>(tid);
            uint32_t d = INVALID_DIGIT;
            if (u < head) d = digit_of(src[u], prm.lo, prm.mask);
            else if (u - head < ntail) d = digit_of(src[tail0 + (u - head)], prm.lo, prm.mask);
            hist_add<K>(hist, d);
        }
        const uint4 *vsrc = reinterpret_cast<const uint4 *>(src + head);
        for (uint32_t vb = 0; vb < nvec; vb += THREADS * U) {
            uint4 w[U];
#pragma unroll
            for (int u = 0; u < U; ++u) {
                uint32_t v = vb + u * THREADS + tid;
                if (v < nvec) w[u] = __ldg(vsrc + v);
            }
#pragma unroll
            for (int u = 0; u < U; ++u) {
                const bool ok = vb + u * THREADS + tid < nvec;
                const K *kk = reinterpret_cast<const K *>(&w[u]);
#pragma unroll
                for (int j = 0; j < VK; ++j) {
                    uint32_t d = ok ? digit_of(kk[j], prm.lo, prm.mask) : INVALID_DIGIT;
                    hist_add<K>(hist, d);
                }
            }
        }
        __syncthreads();
        // ---- decoupled look-back over the tiles of this bucket (tile order = memory order)
        const Bucket bk = prm.buckets[tile.bucket];
        const bool first = t == bk.first_tile;
        const bool lastt = t + 1 == bk.first_tile + bk.ntiles;
        if (tid < RADIX) {
            const S c = hist[tid];
            S *st = status + static_cast<uint64_t>(t) * RADIX + tid;
            S incl;
            if (first) {
                incl = c;
                st_volatile(st, static_cast<S>(SB::INC | c));
            } else {
                st_volatile(st, static_cast<S>(SB::AGG | c));
                S excl = 0;
                const S *q = st - RADIX;
                for (;;) {
                    const S v = ld_volatile(q);
                    if ((v & SB::FLAGS) == 0) continue;  // predecessor not published yet
                    excl += v & SB::VAL;
                    if (v & SB::INC) break;
                    q -= RADIX;
                }
                incl = excl + c;
                st_volatile(st, static_cast<S>(SB::INC | incl));
            }
            if (lastt) tot[tid] = incl;
        }
        if (lastt) {
            __syncthreads();
            classify_bucket<K, S, THREADS>(prm, bk, tile.bucket, tot, scratch);
        }
        __syncthreads();
    }
}

// ------------------------------------------------------------------ stable block rank

// Ranks the KPT keys a warp holds in "warp-striped" order (element e of the block
// = warp * 32 * KPT + c * 32 + lane) by digit, stably: rank = (#elements of smaller
// digit) + (#elements of equal digit earlier in element order).  Result per key:
// the rank of the key within its warp's run of the digit, packed (r << 9) | digit;
// wcnt[w][d] ends up holding the block-wide start of warp w's run of digit d.
//   wcnt: W * NBINS u32, tot: NBINS u32 (shared)
template <int THREADS, int KPT>
__device__ __forceinline__ void warp_rank_walk(uint32_t (&rk)[KPT], uint32_t *mycnt) {
    // on entry rk[c] holds the digit of key c (INVALID_DIGIT for padding lanes)
    const uint32_t ltm = lanemask_lt();
#pragma unroll
    for (int c = 0; c < KPT; ++c) {
        const uint32_t d = rk[c];
        const uint32_t m = __match_any_sync(0xffffffffu, d);
        const uint32_t below = m & ltm;
        const uint32_t pre = mycnt[d];
        __syncwarp();
        if (below == 0) mycnt[d] = pre + __popc(m);
        __syncwarp();
        rk[c] = ((pre + __popc(below)) << 9) | d;
    }
}

// Column scan over warps and exclusive scan over digits: afterwards wcnt[w][d] =
// start of warp w's run of digit d in the block, and tot[d] = start of digit d
// (tot[256] = number of valid elements).
template <int THREADS>
__device__ __forceinline__ void block_rank_scan(uint32_t *wcnt, uint32_t *tot) {
    constexpr int W = THREADS / 32;
    for (int d = threadIdx.x; d < NBINS; d += THREADS) {
        uint32_t run = 0;
#pragma unroll
        for (int w = 0; w < W; ++w) {
            const uint32_t v = wcnt[w * NBINS + d];
            wcnt[w * NBINS + d] = run;
            run += v;
        }
        tot[d] = run;
    }
    __syncthreads();
    warp0_exclusive_scan(tot, NBINS);
    __syncthreads();
    for (int d = threadIdx.x; d < NBINS; d += THREADS) {
        const uint32_t ls = tot[d];
#pragma unroll
        for (int w = 0; w < W; ++w) wcnt[w * NBINS + d] += ls;
    }
}

// ------------------------------------------------------------------ scatter

struct ScatterParams {
    const void *keys_in;
    void *keys_out;
    const void *vals_in;
    void *vals_out;
    int p;
    int lo;
    uint32_t mask;
    const Tile *tiles;
    const Bucket *buckets;
    const void *status;
    const uint32_t *sub_rel;
    void *status_next;  // cleared for pass p+1 (may be NULL)
    int status_bytes;
    Ctl *ctl;
};

template <typename K, typename V, int THREADS, int KPT>
struct ScatterSmem {
    static constexpr int W = THREADS / 32;
    static constexpr int KPB = THREADS * KPT;
    static constexpr size_t off_wcnt = 0;
    static constexpr size_t off_tot = off_wcnt + sizeof(uint32_t) * W * NBINS;
    static constexpr size_t off_gbase = (off_tot + sizeof(uint32_t) * NBINS + 15) & ~size_t(15);
    static constexpr size_t off_keys = off_gbase + sizeof(unsigned long long) * RADIX;
    static constexpr size_t off_vals = (off_keys + sizeof(K) * KPB + 15) & ~size_t(15);
    static constexpr size_t bytes = off_vals + (HasVal<V>::value ? sizeof(V) * KPB : 0);
};

template <typename K, typename V, typename S, int THREADS, int KPT, int MINB>
__global__ void __launch_bounds__(THREADS, MINB) k_scatter(ScatterParams prm) {
    using L = ScatterSmem<K, V, THREADS, KPT>;
    constexpr bool HV = HasVal<V>::value;
    using VT = typename std::conditional<HV, V, uint32_t>::type;
    extern __shared__ __align__(16) unsigned char smem[];
    uint32_t *wcnt = reinterpret_cast<uint32_t *>(smem + L::off_wcnt);
    uint32_t *tot = reinterpret_cast<uint32_t *>(smem + L::off_tot);
    unsigned long long *gbase = reinterpret_cast<unsigned long long *>(smem + L::off_gbase);
    K *skeys = reinterpret_cast<K *>(smem + L::off_keys);
    VT *svals = reinterpret_cast<VT *>(smem + L::off_vals);

    const K *__restrict__ kin = static_cast<const K *>(prm.keys_in);
    K *__restrict__ kout = static_cast<K *>(prm.keys_out);
    const VT *__restrict__ vin = static_cast<const VT *>(prm.vals_in);
    VT *__restrict__ vout = static_cast<VT *>(prm.vals_out);
    const S *status = static_cast<const S *>(prm.status);
    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    const uint32_t wbase = static_cast<uint32_t>(warp) * 32 * KPT;
    const uint32_t T = prm.ctl->ntiles[prm.p];

    for (uint32_t t = blockIdx.x; t < T; t += gridDim.x) {
        const Tile tile = prm.tiles[t];
        const uint32_t count = tile.count;
        S st = 0;
        uint32_t srel = 0;
        if (tid < RADIX) {
            st = status[static_cast<uint64_t>(t) * RADIX + tid];
            srel = prm.sub_rel[static_cast<uint64_t>(tile.bucket) * RADIX + tid];
        }
        const uint64_t boffs = prm.buckets[tile.bucket].offs;
        // ---- load (warp-striped, coalesced)
        K key[KPT];
        VT val[KPT];
        const K *ksrc = kin + tile.offs;
        const VT *vsrc = HV ? vin + tile.offs : nullptr;
#pragma unroll
        for (int c = 0; c < KPT; ++c) {
            const uint32_t e = wbase + c * 32 + lane;
            if (e < count) {
                key[c] = ksrc[e];
                if (HV) val[c] = vsrc[e];
            }
        }
        for (int i = tid; i < (THREADS / 32) * NBINS; i += THREADS) wcnt[i] = 0;
        __syncthreads();
        // ---- stable rank
        uint32_t rk[KPT];
        if (wbase < count) {
#pragma unroll
            for (int c = 0; c < KPT; ++c) {
                const uint32_t e = wbase + c * 32 + lane;
                rk[c] = e < count ? digit_of(key[c], prm.lo, prm.mask) : INVALID_DIGIT;
            }
            warp_rank_walk<THREADS, KPT>(rk, wcnt + warp * NBINS);
        }
        __syncthreads();
        block_rank_scan<THREADS>(wcnt, tot);
        if (tid < RADIX) {
            // destination of smem slot j holding digit d: gbase[d] + j
            const uint64_t incl = static_cast<uint64_t>(st & StatusBits<S>::VAL);
            gbase[tid] = boffs + srel + incl - tot[tid + 1];
        }
        __syncthreads();
        // ---- stage in shared memory at the rank
        if (wbase < count) {
            const uint32_t *mycnt = wcnt + warp * NBINS;
#pragma unroll
            for (int c = 0; c < KPT; ++c) {
                const uint32_t d = rk[c] & 511u;
                if (d != INVALID_DIGIT) {
                    const uint32_t r = mycnt[d] + (rk[c] >> 9);
                    skeys[r] = key[c];
                    if (HV) svals[r] = val[c];
                }
            }
        }
        __syncthreads();
        // ---- write-combined stores: consecutive slots of a digit run are consecutive addresses
#pragma unroll
        for (int c = 0; c < KPT; ++c) {
            const uint32_t j = c * THREADS + tid;
            if (j < count) {
                const K k = skeys[j];
                const uint64_t pos = gbase[digit_of(k, prm.lo, prm.mask)] + j;
                kout[pos] = k;
                if (HV) vout[pos] = svals[j];
            }
        }
        __syncthreads();
    }
    // clear the look-back status of pass p+1 (the array pass p-1 used)
    if (prm.status_next) {
        const uint64_t words16 =
            (static_cast<uint64_t>(prm.ctl->ntiles[prm.p + 1]) * RADIX * prm.status_bytes) / 16;
        uint4 *s = static_cast<uint4 *>(prm.status_next);
        for (uint64_t i = static_cast<uint64_t>(blockIdx.x) * THREADS + tid; i < words16;
             i += static_cast<uint64_t>(gridDim.x) * THREADS)
            s[i] = make_uint4(0, 0, 0, 0);
    }
}

// ------------------------------------------------------------------ local sort

struct LocalParams {
    const void *src_keys[3];  // indexed by SrcCode
    const void *src_vals[3];
    void *keys_out;
    void *vals_out;
    const LocalEntry *list;
    const uint32_t *count;  // entries in the list
    int begin_bit;
};

template <typename K, typename V, int THREADS, int KPT>
struct LocalSmem {
    static constexpr int W = THREADS / 32;
    static constexpr int CAP = THREADS * KPT;
    static constexpr size_t off_wcnt = 0;
    static constexpr size_t off_tot = off_wcnt + sizeof(uint32_t) * W * NBINS;
    static constexpr size_t off_red = (off_tot + sizeof(uint32_t) * NBINS + 15) & ~size_t(15);
    static constexpr size_t off_keys = off_red + sizeof(K) * 2 * W;
    static constexpr size_t off_vals = (off_keys + sizeof(K) * CAP + 15) & ~size_t(15);
    static constexpr size_t bytes = off_vals + (HasVal<V>::value ? sizeof(V) * CAP : 0);
};

template <typename K>
__device__ __forceinline__ K warp_and(K x) {
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) x &= __shfl_xor_sync(0xffffffffu, x, o);
    return x;
}
template <typename K>
__device__ __forceinline__ K warp_or(K x) {
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) x |= __shfl_xor_sync(0xffffffffu, x, o);
    return x;
}

template <typename K, typename V, int THREADS, int KPT, int MINB>
__global__ void __launch_bounds__(THREADS, MINB) k_local(LocalParams prm) {
    using L = LocalSmem<K, V, THREADS, KPT>;
    constexpr int W = THREADS / 32;
    constexpr bool HV = HasVal<V>::value;
    using VT = typename std::conditional<HV, V, uint32_t>::type;
    extern __shared__ __align__(16) unsigned char smem[];
    uint32_t *wcnt = reinterpret_cast<uint32_t *>(smem + L::off_wcnt);
    uint32_t *tot = reinterpret_cast<uint32_t *>(smem + L::off_tot);
    K *red = reinterpret_cast<K *>(smem + L::off_red);
    K *skeys = reinterpret_cast<K *>(smem + L::off_keys);
    VT *svals = reinterpret_cast<VT *>(smem + L::off_vals);
    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    const uint32_t wbase = static_cast<uint32_t>(warp) * 32 * KPT;
    const uint32_t nent = *prm.count;
    K *__restrict__ kout = static_cast<K *>(prm.keys_out);
    VT *__restrict__ vout = static_cast<VT *>(prm.vals_out);

    for (uint32_t ei = blockIdx.x; ei < nent; ei += gridDim.x) {
        const LocalEntry en = prm.list[ei];
        const uint32_t count = en.count;
        // select without dynamic indexing of the parameter arrays (keeps them out of local memory)
        const void *kbase = en.src == SRC_IN ? prm.src_keys[SRC_IN]
                            : en.src == SRC_AUX ? prm.src_keys[SRC_AUX] : prm.src_keys[SRC_OUT];
        const void *vbase = en.src == SRC_IN ? prm.src_vals[SRC_IN]
                            : en.src == SRC_AUX ? prm.src_vals[SRC_AUX] : prm.src_vals[SRC_OUT];
        const K *ksrc = static_cast<const K *>(kbase) + en.offs;
        const VT *vsrc = HV ? static_cast<const VT *>(vbase) + en.offs : nullptr;
        K key[KPT];
        VT val[KPT];
        K a = ~K(0), o = K(0);
#pragma unroll
        for (int c = 0; c < KPT; ++c) {
            const uint32_t e = wbase + c * 32 + lane;
            if (e < count) {
                key[c] = ksrc[e];
                if (HV) val[c] = vsrc[e];
                a &= key[c];
                o |= key[c];
            }
        }
        // bits that vary across the bucket: digits where they are all equal are skipped
        a = warp_and(a);
        o = warp_or(o);
        if (lane == 0) {
            red[warp] = a;
            red[W + warp] = o;
        }
        __syncthreads();
        K diff = 0;
        {
            K aa = ~K(0), oo = K(0);
#pragma unroll
            for (int w = 0; w < W; ++w) {
                aa &= red[w];
                oo |= red[W + w];
            }
            diff = aa ^ oo;
        }
        bool moved = false;
        for (int lo = prm.begin_bit; lo < en.hi_bit; lo += 8) {
            const int width = min(8, en.hi_bit - lo);
            const uint32_t mask = (1u << width) - 1u;
            if ((static_cast<uint32_t>(diff >> lo) & mask) == 0) continue;  // constant digit: identity pass
            moved = true;
            for (int i = tid; i < W * NBINS; i += THREADS) wcnt[i] = 0;
            __syncthreads();
            uint32_t rk[KPT];
            if (wbase < count) {
#pragma unroll
                for (int c = 0; c < KPT; ++c) {
                    const uint32_t e = wbase + c * 32 + lane;
                    rk[c] = e < count ? digit_of(key[c], lo, mask) : INVALID_DIGIT;
                }
                warp_rank_walk<THREADS, KPT>(rk, wcnt + warp * NBINS);
            }
            __syncthreads();
            block_rank_scan<THREADS>(wcnt, tot);
            __syncthreads();
            if (wbase < count) {
                const uint32_t *mycnt = wcnt + warp * NBINS;
#pragma unroll
                for (int c = 0; c < KPT; ++c) {
                    const uint32_t d = rk[c] & 511u;
                    if (d != INVALID_DIGIT) {
                        const uint32_t r = mycnt[d] + (rk[c] >> 9);
                        skeys[r] = key[c];
                        if (HV) svals[r] = val[c];
                    }
                }
            }
            __syncthreads();
#pragma unroll
            for (int c = 0; c < KPT; ++c) {
                const uint32_t e = wbase + c * 32 + lane;
                if (e < count) {
                    key[c] = skeys[e];
                    if (HV) val[c] = svals[e];
                }
            }
            __syncthreads();
        }
        if (moved || en.src != SRC_OUT) {
#pragma unroll
            for (int c = 0; c < KPT; ++c) {
                const uint32_t e = wbase + c * 32 + lane;
                if (e < count) {
                    kout[en.offs + e] = key[c];
                    if (HV) vout[en.offs + e] = val[c];
                }
            }
        }
        __syncthreads();  // red[] reuse
    }
}

}  // namespace hrs
