// hrs_device.cuh -- sm_100a kernels of the stable hybrid MSD radix sort.
//
// Paper: Stehle & Jacobsen, arXiv 1611.01137 (PAPER.md lines cited as P:<line>).
// Every pass p of the MSD recursion (Fig 1) runs three kernels over a
// device-resident bucket table whose buckets are cut into tiles ("key blocks",
// P:517-541), so each pass costs a constant number of launches and the host never
// reads device memory:
//
//   k_hist<p>      reads the keys of every tile straight from global memory in 16-byte
//                  vectors and counts the digit into one block histogram per tile with
//                  plain shared-memory atomics (on B200 they run at full HBM
//                  read rate even for a constant digit -- profiles/r01_micro_hist.txt --
//                  so neither warp aggregation nor the paper's sorting-network thread
//                  reduction, is needed).  Each CTA owns a contiguous run of
//                  tiles, records each tile's prefix within its bucket segment and adds
//                  the bucket histograms to global memory once per bucket run.
//   k_classify<p>  one CTA per bucket: exclusive prefix sum of the bucket histogram
//                  into sub-bucket offsets and classification of the
//                  sub-buckets (R1-R3 P:805-811, merging P:552-561) into next-pass
//                  buckets/tiles and local-sort lists; 8 more CTAs scan the CTA runs
//                  into per-run carries.
//   k_scatter<p>   per tile, with the next tile's keys already in flight through TMA: a
//                  STABLE in-tile rank (per-warp digit counters), staging in shared
//                  memory and write-combined stores of every digit run (P:704-722,
//                  Fig 3); values follow their keys.  The tile-ordered
//                  offset of every tile inside its sub-bucket is known before the
//                  scatter starts (k_hist prefixes + k_classify carries): deterministic,
//                  no look-back, and it replaces the atomicAdd chunk reservation of
//                  P:696-703 (which is not stable).
//
// then the buckets of at most ∂ˆ records are sorted on chip, one launch per size class
// (P:562-577): the two largest classes by k_local_cnt (one counting sort on the top
// varying sort bits, ties ordered afterwards), the others -- and every bucket the
// counting sort hands off -- by k_local, a stable LSD radix sort of (key, index)
// composites over the remaining bits that skips digits constant across the
// bucket and gathers the values once at the end.
//
// Stability everywhere (ties keep input order) is the one deliberate departure
// from the paper: the output is the unique stable sort.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

#include <type_traits>

#include "../../include/hrs.h"

#ifndef HRS_EXP
#define HRS_EXP 0  // kernel-variant experiments (micro/scatter_exp.py); 0 in the product
#endif
#ifndef HRS_WAIT1
#define HRS_WAIT1 0  // (measured slower when 1) k_hist / k_scatter: one warp waits on the TMA mbarrier, a CTA barrier releases the others
#endif
#ifndef HRS_WIDE64
#define HRS_WIDE64 1  // measured: c4 AND-2/3/4 -4 to -9 %, uniform unchanged
#endif
#ifndef HRS_WO_UNROLL
#define HRS_WO_UNROLL 4
#endif
namespace hrs { constexpr int WO_UNROLL = HRS_WO_UNROLL; }
#ifndef HRS_SC_STHINT
#define HRS_SC_STHINT 0  // measured: evict_last stores on pass 1 only slow pass 2 (0.99 -> 1.08 ms), on every pass no change
#endif
#ifndef HRS_SC_VSPLIT
#define HRS_SC_VSPLIT 1  // one value staging buffer (two key buffers): larger tiles (0: two of each)
#endif
#ifndef HRS_SC_DIRECT
#define HRS_SC_DIRECT 0  // experiment: values placed from registers, no slot index, no stability check
#endif
#ifndef HRS_RANK2
#define HRS_RANK2 1  // Ranker::rank2 for blocks of >= 256 threads
#endif

namespace hrs {

constexpr int RADIX = 256;
constexpr int NBINS = 257;  // 256 digit values + 1 bin for padding lanes
constexpr uint32_t INVALID_DIGIT = 256;
constexpr uint64_t CTL_MAGIC = 0x4852535f31363131ull;  // "HRS_1611"

enum SrcCode : uint16_t { SRC_IN = 0, SRC_AUX = 1, SRC_OUT = 2 };

// A bucket that is counting-sorted in the current pass.  Its tiles ("key blocks",
// P:521-524; up to KPB consecutive records each) are first_tile .. first_tile +
// ntiles - 1, consecutive and in memory order: that order makes the pass stable.
struct Bucket {
    uint64_t offs;
    uint32_t count;
    uint32_t first_tile;
    uint32_t ntiles;
    uint16_t src;   // SrcCode of the buffer holding the bucket's records at the start of the pass
    uint16_t skip;  // set by k_classify: the digit is constant over the bucket and it never
                    // moved (src == SRC_IN): k_scatter leaves its records where they are
};
// One tile as k_hist saw it, for k_scatter: records [offs, offs + count) of bucket
// `bucket`; carry_row = the hist CTA whose carry applies (tile in the first bucket
// segment of that CTA's run), or EMPTY.
struct TileDesc {
    uint64_t offs;
    uint32_t count;
    uint32_t bucket;
    uint32_t carry_row;
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
    // tiles (high 32 bits) and buckets (low 32 bits) of pass p (1-based), allocated
    // together by one 64-bit atomic so bucket order == tile order
    unsigned long long alloc[HRS_MAX_PASSES + 2];
    uint32_t nlocal[HRS_NUM_CLASSES];       // entries in local list c
    uint32_t claim[HRS_MAX_PASSES + 2];     // k_scatter tile claims of pass p
    uint32_t nlocal_wide[HRS_NUM_CLASSES];  // entries the narrow local sort handed to the wide one, per configuration
    uint32_t nlocal_fb2;                    // entries the counting local sort handed to the narrow one
    uint32_t overflow;
    uint32_t pad_;
    unsigned long long recs_in_pass[HRS_MAX_PASSES + 2];
    unsigned long long local_recs;
    unsigned long long merged_groups;
    unsigned long long redo;  // blocks that redid a tile / bucket with the stable-by-construction rank
    unsigned long long skipped_in_pass[HRS_MAX_PASSES + 2];  // records of skipped buckets (no scatter)
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

struct NoVal {};
template <typename V>
struct HasVal {
    static constexpr bool value = true;
};
template <>
struct HasVal<NoVal> {
    static constexpr bool value = false;
};
template <typename V>
using ValT = typename std::conditional<HasVal<V>::value, V, uint32_t>::type;

// Local-sort size classes (P:562-566 gives [1,128], (128,256], (256,512], ... as an
// example): powers of two up to 4096, then (4096, 4608] and (4608, 8192] so that the
// ~4096-record buckets a uniform input leaves after two passes keep every warp busy.
__host__ __device__ __forceinline__ uint32_t class_capacity(int c) {
    return c < 6 ? (128u << c) : (c == 6 ? 4608u : 8192u);
}
__host__ __device__ __forceinline__ int size_class_of(uint32_t size) {
    int c = 0;
    while (class_capacity(c) < size && c < HRS_NUM_CLASSES - 1) ++c;
    return c;
}

__host__ __device__ constexpr size_t align16(size_t x) { return (x + 15) & ~size_t(15); }

// The configuration (size class) of the wide local sort that takes a hand-off of size
// class c: 1024 records (class 3) for small ones, 2048 (class 4), else the largest --
// except for 64-bit keys (mid = 1), where classes 5 and 6 keep their own configuration
// (4096 / 4608 records): measured on B200, c4 AND-2 16.39 -> 15.58 ms, AND-3 17.33 ->
// 16.71 ms, uniform unchanged; for 32-bit keys the two extra launches only cost latency
// (2^20 keys-only 90.8 -> 96.2 us), so they keep the largest.
#ifndef HRS_WIDE_MID
#define HRS_WIDE_MID 1
#endif
__host__ __device__ __forceinline__ int wide_cfg(int c, int top, bool mid) {
    return c <= 3 ? 3 : (c == 4 ? 4 : (HRS_WIDE_MID && mid ? (c < top ? c : top) : top));
}

// Exclusive scan of n <= 288 u32 values in shared memory, in place, by warp 0.
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

// ------------------------------------------------------------------ tiles derived from the bucket table

__device__ __forceinline__ uint32_t alloc_tiles(unsigned long long a) { return static_cast<uint32_t>(a >> 32); }
__device__ __forceinline__ uint32_t alloc_buckets(unsigned long long a) { return static_cast<uint32_t>(a); }

// Tile t of a pass belongs to the bucket b with first_tile <= t < first_tile + ntiles;
// bucket ids are allocated in tile order, so a binary search finds it.
__device__ __forceinline__ uint32_t find_bucket(const Bucket *bks, uint32_t nb, uint32_t t) {
    uint32_t lo = 0, hi = nb - 1;
    while (lo < hi) {
        const uint32_t mid = (lo + hi + 1) >> 1;
        if (bks[mid].first_tile <= t) lo = mid;
        else hi = mid - 1;
    }
    return lo;
}

// Walks the tiles [tb, te) of one CTA in order (used by the producer thread).
struct TileCursor {
    const Bucket *bks;
    uint32_t t, te, b, k;
    Bucket bk;
    uint32_t kpb;
    __device__ __forceinline__ void start(const Bucket *bks_, uint32_t nb, uint32_t tb, uint32_t te_, uint32_t kpb_) {
        bks = bks_;
        t = tb;
        te = te_;
        kpb = kpb_;
        if (t < te) {
            b = find_bucket(bks, nb, t);
            bk = bks[b];
            k = t - bk.first_tile;
        }
    }
    __device__ __forceinline__ bool valid() const { return t < te; }
    __device__ __forceinline__ uint64_t offs() const { return bk.offs + static_cast<uint64_t>(k) * kpb; }
    __device__ __forceinline__ uint32_t count() const { return min(kpb, bk.count - k * kpb); }
    __device__ __forceinline__ bool last_of_bucket() const { return k + 1 == bk.ntiles; }
    __device__ __forceinline__ void next() {
        ++t;
        if (t >= te) return;
        if (++k == bk.ntiles) {
            ++b;
            bk = bks[b];
            k = 0;
        }
    }
};

// Per-CTA range bookkeeping shared by k_hist, k_classify and k_scatter (same grid):
// the digit counts of the CTA's last bucket segment and the bucket ids of its first
// and last tile; k_classify turns them into the carry of each CTA's first segment.
constexpr uint32_t EMPTY_RANGE = 0xFFFFFFFFu;
struct RangeMeta {
    uint32_t first_bucket, last_bucket;
};

__host__ __device__ __forceinline__ uint32_t range_begin(uint32_t T, uint32_t c, uint32_t G) {
    return static_cast<uint32_t>((static_cast<uint64_t>(T) * c) / G);
}

// Programmatic dependent launch: every kernel of a sort is launched with PDL, so its
// launch and prologue overlap the previous kernel's tail; it waits here before it
// touches memory the previous kernels wrote.
// With HRS_PDL_EARLY the kernel first lets its dependent grid launch (its CTAs then wait
// here for this grid's completion and memory flush, so early triggering is safe).
#ifndef HRS_PDL_EARLY
#define HRS_PDL_EARLY 0  // measured: no gain at 2^20, c2 +2 %
#endif
__device__ __forceinline__ void pdl_wait() {
    if (HRS_PDL_EARLY) asm volatile("griddepcontrol.launch_dependents;" ::: "memory");
    asm volatile("griddepcontrol.wait;" ::: "memory");
}

// ------------------------------------------------------------------ TMA bulk copies (cp.async.bulk + mbarrier)

__device__ __forceinline__ uint32_t smem_u32(const void *p) {
    return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}
__device__ __forceinline__ void mbar_init(uint64_t *bar, uint32_t count) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count) : "memory");
}
__device__ __forceinline__ void mbar_fence_init() {
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
}
__device__ __forceinline__ void fence_proxy_async() {
    asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
}
__device__ __forceinline__ void mbar_arrive_expect_tx(uint64_t *bar, uint32_t bytes) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes)
                 : "memory");
}
__device__ __forceinline__ void mbar_arrive(uint64_t *bar) {
    asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(bar)) : "memory");
}
// HRS_MBAR_HINT (ns): the suspend-time hint of the try_wait -- a waiting thread sleeps until
// the phase completes or the hint elapses instead of re-polling (0: the default time limit)
#ifndef HRS_MBAR_HINT
#define HRS_MBAR_HINT 0  // measured: 1 us and 100 us hints change nothing (c2, AND-2)
#endif
__device__ __forceinline__ void mbar_wait(uint64_t *bar, uint32_t parity) {
#if HRS_MBAR_HINT
    asm volatile(
        "{\n"
        ".reg .pred P1;\n"
        "HRS_WAIT_%=:\n"
        "mbarrier.try_wait.parity.shared::cta.b64 P1, [%0], %1, %2;\n"
        "@!P1 bra HRS_WAIT_%=;\n"
        "}\n" ::"r"(smem_u32(bar)),
        "r"(parity), "n"(HRS_MBAR_HINT)
        : "memory");
#else
    asm volatile(
        "{\n"
        ".reg .pred P1;\n"
        "HRS_WAIT_%=:\n"
        "mbarrier.try_wait.parity.shared::cta.b64 P1, [%0], %1;\n"
        "@!P1 bra HRS_WAIT_%=;\n"
        "}\n" ::"r"(smem_u32(bar)),
        "r"(parity)
        : "memory");
#endif
}
__device__ __forceinline__ uint64_t policy_evict_first() {
    uint64_t p;
    asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(p));
    return p;
}
__device__ __forceinline__ uint64_t policy_evict_last() {
    uint64_t p;
    asm volatile("createpolicy.fractional.L2::evict_last.b64 %0, 1.0;" : "=l"(p));
    return p;
}
// 4-byte global store with an L2 cache-eviction hint
__device__ __forceinline__ void st_hint(uint32_t *p, uint32_t v, uint64_t pol) {
    asm volatile("st.global.L2::cache_hint.b32 [%0], %1, %2;" ::"l"(p), "r"(v), "l"(pol) : "memory");
}
__device__ __forceinline__ void bulk_g2s(void *dst, const void *src, uint32_t bytes, uint64_t *bar, uint64_t pol) {
    asm volatile(
        "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes.L2::cache_hint [%0], [%1], %2, [%3], %4;" ::
            "r"(smem_u32(dst)),
        "l"(src), "r"(bytes), "r"(smem_u32(bar)), "l"(pol)
        : "memory");
}
// 16-byte asynchronous copy global -> shared (a work-list entry fetched ahead of its use)
__device__ __forceinline__ void cp_async16(void *dst, const void *src) {
    asm volatile("cp.async.ca.shared.global [%0], [%1], 16;\ncp.async.commit_group;" ::"r"(smem_u32(dst)), "l"(src)
                 : "memory");
}
__device__ __forceinline__ void cp_async_wait_all() { asm volatile("cp.async.wait_all;" ::: "memory"); }

// A staged segment of `count` elements starting at global `src`, inside a buffer
// [base, limit): one bulk copy moves the 16-byte aligned SUPERSET of the segment (up to
// 12 bytes of the neighbouring segments on each side, which are never used), clipped
// to the buffer, so the unaligned head and tail need no separate global loads.  Element
// i lives in shared memory at sbuf[pad + i] for i in [i0, i1) (i0 <= 0 and i1 >= count
// unless the clip to the buffer cut the copy); elements outside stay in global memory.
// The staging buffer needs room for count + 2 * 16 / sizeof(T) elements.
struct Seg {
    uint32_t pad;
    int32_t i0, i1;
};
template <typename T>
__device__ __forceinline__ uint32_t seg_plan(const T *src, uint32_t count, const T *base, const T *limit, Seg &sg) {
    const uintptr_t a = reinterpret_cast<uintptr_t>(src);
    sg.pad = static_cast<uint32_t>((a & 15) / sizeof(T));
    uintptr_t lo = a & ~uintptr_t(15);
    const uintptr_t b16 = (reinterpret_cast<uintptr_t>(base) + 15) & ~uintptr_t(15);
    if (lo < b16) lo = b16;
    uintptr_t hi = (a + static_cast<uintptr_t>(count) * sizeof(T) + 15) & ~uintptr_t(15);
    const uintptr_t l16 = reinterpret_cast<uintptr_t>(limit) & ~uintptr_t(15);
    if (hi > l16) hi = l16;
    if (count > 0 && hi > lo) {
        sg.i0 = static_cast<int32_t>((static_cast<intptr_t>(lo) - static_cast<intptr_t>(a)) / static_cast<intptr_t>(sizeof(T)));
        sg.i1 = static_cast<int32_t>((static_cast<intptr_t>(hi) - static_cast<intptr_t>(a)) / static_cast<intptr_t>(sizeof(T)));
        return static_cast<uint32_t>(hi - lo);
    }
    sg.i0 = sg.i1 = 0;
    return 0;
}
template <typename T>
__device__ __forceinline__ void seg_issue(T *sbuf, const T *src, const Seg &sg, uint64_t *bar, uint64_t pol) {
    if (sg.i1 > sg.i0)
        bulk_g2s(sbuf + (static_cast<int32_t>(sg.pad) + sg.i0), src + sg.i0,
                 static_cast<uint32_t>(sg.i1 - sg.i0) * static_cast<uint32_t>(sizeof(T)), bar, pol);
}
// every element of the segment is in shared memory
__device__ __forceinline__ bool seg_full(const Seg &sg, uint32_t count) {
    return sg.i0 <= 0 && sg.i1 >= static_cast<int32_t>(count);
}
template <typename T>
__device__ __forceinline__ T seg_get(const T *sbuf, const T *src, const Seg &sg, uint32_t i) {
    return (static_cast<int32_t>(i) >= sg.i0 && static_cast<int32_t>(i) < sg.i1) ? sbuf[sg.pad + i] : src[i];
}
// copy the elements the bulk copy did not cover into the staging buffer, so
// sbuf[pad + i] is valid for all i < count (only segments at the ends of the buffer)
template <typename T, int THREADS>
__device__ __forceinline__ void seg_fill_edges(T *sbuf, const T *src, const Seg &sg, uint32_t count) {
    if (seg_full(sg, count)) return;
    const uint32_t h = sg.i1 > sg.i0 ? static_cast<uint32_t>(max(sg.i0, 0)) : count;     // head [0, h)
    const uint32_t t = sg.i1 > sg.i0 ? static_cast<uint32_t>(min(sg.i1, static_cast<int32_t>(count))) : count;  // tail [t, count)
    for (uint32_t j = threadIdx.x; j < h + (count - t); j += THREADS) {
        const uint32_t i = j < h ? j : t + (j - h);
        sbuf[sg.pad + i] = src[i];
    }
}

// ------------------------------------------------------------------ stable block rank
//
// The keys a warp holds are in "warp-striped" order (element e of the tile is
// warp * 32 * kpt + c * 32 + lane).  The stable rank of a key (its slot among all
// keys of the tile, ties in element order) is
//     start[d] + (keys of digit d in earlier warps) + (keys of digit d before it in its warp),
// computed in three steps:
//   1. count: per-warp digit counters in shared memory, one atomic per key;
//   2. scan: exclusive prefix over the warps per digit and over the digits, folded
//      into each warp's counters = first slot of the warp's run of each digit;
//   3. in-warp rank, one of two ways, chosen per warp:
//      fast  -- the count atomics of step 1 RETURN the old counter value, and that is
//               taken as the in-warp rank.  It is the stable rank exactly when the
//               same-address lanes of one atomic instruction are served in lane order
//               (and a warp's instructions in program order), which B200 does
//               (profiles/r01_micro_rank_ballot.txt) but PTX leaves unspecified, so
//               every caller checks the order it produced and redoes the tile with
//               the exact path if it is not the stable one.  One shared operation
//               per key besides the count.
//      exact -- stable by construction: column by column, every lane reads the warp's
//               next free slot of its digit, adds 1 with a non-returning atomic and
//               reads the counter back; the difference is the number of lanes of the
//               column with that digit, and lanes with duplicates take their order
//               from one match-any over the column where all other lanes share one
//               dummy value (match-any over 32 distinct values is what makes a pure
//               match-based multisplit slow on B200; profiles/r01_micro_rank.txt).
//   Returning atomics serialise same-address lanes, so a warp whose first column shows
//   heavy digit contention (skewed keys) takes the exact path, where same-address
//   lanes are cheap.
template <int THREADS, int KPT>
struct Ranker {
    static constexpr int W = THREADS / 32;
    static constexpr size_t cnt_words = static_cast<size_t>(W) * NBINS;
    static constexpr size_t smem_bytes = sizeof(uint32_t) * (cnt_words + 2 * 288);
    static_assert(32 * KPT < (1 << 16), "the in-warp rank is packed above the digit");
    uint32_t *cnt;    // [W][NBINS]
    uint32_t *tot;    // [288] digit totals of the tile
    uint32_t *start;  // [288] first slot of each digit (valid after the caller's next barrier)

    __device__ __forceinline__ uint32_t *vcnt(int w) const { return cnt + w * NBINS; }

    // THREADS >= 256: the per-digit fold is done by one thread per digit (see rank2)
    static constexpr bool FOLD = THREADS >= RADIX && HRS_RANK2;
    static constexpr int BOWN = THREADS > RADIX ? RADIX : 0;  // thread that folds bin 256

    __device__ __forceinline__ void init(uint32_t *base) {
        cnt = base;
        tot = base + cnt_words;
        start = tot + 288;
        for (int i = threadIdx.x; i < static_cast<int>(cnt_words); i += THREADS) cnt[i] = 0;
    }

    // the fold for THREADS >= 256 after the count phase and its barrier: thread d (< 256)
    // reads the W warp counters of digit d, scans the digit totals with shuffles and
    // writes every warp's first slot of digit d back (rank() instead has every warp
    // re-read the 257 totals and fold them into its own counters).  About 60 % of the
    // per-digit shared-memory traffic of rank(), one more barrier.
    __device__ __forceinline__ void fold2(uint2 *gs) {
        const int tid = threadIdx.x, warp = tid >> 5, lane = tid & 31;
        uint32_t *wsum = tot;  // [8] digit totals of warps 0..7
        uint32_t t = 0;
        if (tid < RADIX) {
#pragma unroll
            for (int w = 0; w < W; ++w) t += vcnt(w)[tid];
            uint32_t incl = t;
#pragma unroll
            for (int o = 1; o < 32; o <<= 1) {
                const uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
                if (lane >= o) incl += y;
            }
            if (lane == 31) wsum[warp] = incl;
            t = incl - t;  // exclusive within the warp's 32 digits
        }
        __syncthreads();
        if (tid < RADIX) {
            uint32_t run = t;
#pragma unroll
            for (int w = 0; w < RADIX / 32; ++w) run += w < warp ? wsum[w] : 0u;
            if (gs != nullptr) gs[tid] = make_uint2(gs[tid].x - run, run);
#pragma unroll
            for (int w = 0; w < W; ++w) {  // (counts re-read: fewer live registers across the barrier)
                const uint32_t nw = vcnt(w)[tid];
                vcnt(w)[tid] = run;
                run += nw;
            }
        }
        if (tid == BOWN) {  // bin 256 (padding lanes): after every digit
            uint32_t run = 0;
#pragma unroll
            for (int w = 0; w < RADIX / 32; ++w) run += wsum[w];
            for (int w = 0; w < W; ++w) {
                const uint32_t nw = vcnt(w)[RADIX];
                vcnt(w)[RADIX] = run;
                run += nw;
            }
        }
        __syncthreads();
    }

    // in-warp ranks from the folded counters (warp-local; clears the warp's counters)
    __device__ __forceinline__ void lookup(uint32_t (&dg)[KPT], int kpt, bool active, uint32_t ltm, bool fast) {
        const int lane = threadIdx.x & 31;
        uint32_t *ca = vcnt(threadIdx.x >> 5);
        if (active) {
            if (fast) {
#pragma unroll
                for (int c = 0; c < KPT; ++c)
                    if (c < kpt) dg[c] = ca[dg[c] & 0xFFFFu] + (dg[c] >> 16);
            } else {
#pragma unroll
                for (int c = 0; c < KPT; ++c) {
                    const bool v0 = c < kpt;
                    const uint32_t d0 = v0 ? dg[c] : 0u;
                    const uint32_t p0 = v0 ? ca[d0] : 0u;
                    __syncwarp();
                    if (v0) atomicAdd(&ca[d0], 1u);
                    __syncwarp();
                    const uint32_t k0 = v0 ? ca[d0] - p0 : 0u;
                    const uint32_t m = __match_any_sync(0xffffffffu, k0 > 1 ? d0 : 0xFFFFFFFFu);
                    if (v0) dg[c] = p0 + (k0 > 1 ? __popc(m & ltm) : 0u);
                }
            }
        }
        __syncwarp();
        for (int d = lane; d < NBINS; d += 32) ca[d] = 0;
    }

    __device__ __forceinline__ void rank(uint32_t (&dg)[KPT], int kpt, bool active, uint32_t ltm, bool allow_fast,
                                         uint2 *gs = nullptr) {
        const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
        uint32_t *ca = vcnt(warp);
        bool fast = false;
        if (active && allow_fast) {
            // contention probe: equal digits among the 5 butterfly partners of column 0
            // (a uniform digit gives 0.6 on average over the warp)
            const uint32_t d0 = dg[0];
            uint32_t eq = 0;
#pragma unroll
            for (int k = 1; k < 32; k <<= 1) eq += __shfl_xor_sync(0xffffffffu, d0, k) == d0;
            fast = __reduce_add_sync(0xffffffffu, eq) < 8;
        }
        if (active) {
            if (fast) {
#pragma unroll
                for (int c = 0; c < KPT; ++c)
                    if (c < kpt) dg[c] |= atomicAdd(&ca[dg[c]], 1u) << 16;
            } else {
#pragma unroll
                for (int c = 0; c < KPT; ++c)
                    if (c < kpt) atomicAdd(&ca[dg[c]], 1u);
            }
        }
        if constexpr (FOLD) {
            // a block where some warp takes the exact rank (skewed digits) folds with one
            // thread per digit (measured faster there); otherwise every warp folds its own
            if (__syncthreads_or(active && !fast)) {
                fold2(gs);
                lookup(dg, kpt, active, ltm, fast);
                return;
            }
        } else {
            __syncthreads();
        }
        // exclusive prefix over the warps per digit, digit totals
        for (int d = threadIdx.x; d < NBINS; d += THREADS) {
            uint32_t v[W];
#pragma unroll
            for (int w = 0; w < W; ++w) v[w] = vcnt(w)[d];
            uint32_t run = 0;
#pragma unroll
            for (int w = 0; w < W; ++w) {
                vcnt(w)[d] = run;
                run += v[w];
            }
            tot[d] = run;
        }
        __syncthreads();
        // every warp scans the 257 digit totals itself (lane l: digits 9l .. 9l+8) and
        // folds the digit starts into its own counters -- no barrier for a single-warp
        // scan; warp 0 also publishes the starts (read by the caller after its next barrier)
        {
            constexpr int PER = 9;
            uint32_t v[PER];
            uint32_t sum = 0;
#pragma unroll
            for (int i = 0; i < PER; ++i) {
                const int d = lane * PER + i;
                v[i] = d < NBINS ? tot[d] : 0u;
                sum += v[i];
            }
            uint32_t incl = sum;
#pragma unroll
            for (int o = 1; o < 32; o <<= 1) {
                const uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
                if (lane >= o) incl += y;
            }
            uint32_t run = incl - sum;
#pragma unroll
            for (int i = 0; i < PER; ++i) {
                const int d = lane * PER + i;
                if (d < NBINS) {
                    ca[d] += run;
                    if (warp == 0) {
                        start[d] = run;
                        if (gs != nullptr && d < RADIX) gs[d] = make_uint2(gs[d].x - run, run);
                    }
                }
                run += v[i];
            }
        }
        __syncwarp();
        lookup(dg, kpt, active, ltm, fast);
    }
};

// ------------------------------------------------------------------ init / copy

struct InitParams {
    Ctl *ctl;
    Bucket *buckets;         // pass-1 bucket table
    uint32_t *tot;           // pass-1 bucket histograms (row 0 is cleared)
    LocalEntry *root_local;  // list of the root's size class (n <= ∂ˆ)
    int root_class;
    uint64_t n;
    uint32_t kpb;
    int counting;  // 1: the root bucket is counting-sorted
    int end_bit;
    uint32_t key_bytes, value_bytes;
    // hrs_sort_grouped: the input is already grouped by the first digit with these counts
    // (2^width u64): pass 1's partition is given, its histogram is this, it moves nothing
    const uint64_t *grouped_hist;
    uint32_t grouped_radix;
};

static __global__ void k_init(InitParams prm) {
    pdl_wait();
    const uint64_t n = prm.n;
    const uint32_t T1 = prm.counting ? static_cast<uint32_t>((n + prm.kpb - 1) / prm.kpb) : 0u;
    if (blockIdx.x == 0) {
        uint32_t *w = reinterpret_cast<uint32_t *>(prm.ctl);
        for (int i = threadIdx.x; i < static_cast<int>(sizeof(Ctl) / 4); i += blockDim.x) w[i] = 0;
        if (prm.counting)
            for (int i = threadIdx.x; i < RADIX; i += blockDim.x)
                prm.tot[i] = (prm.grouped_hist && static_cast<uint32_t>(i) < prm.grouped_radix)
                                 ? static_cast<uint32_t>(prm.grouped_hist[i])
                                 : 0u;
        __syncthreads();
        if (threadIdx.x == 0) {
            Ctl *c = prm.ctl;
            c->magic = CTL_MAGIC;
            c->n = n;
            c->key_bytes = prm.key_bytes;
            c->value_bytes = prm.value_bytes;
            if (prm.counting) {
                // (grouped input: pass 1 has its bucket but no tiles and moves no record)
                c->alloc[1] = (static_cast<unsigned long long>(prm.grouped_hist ? 0u : T1) << 32) | 1ull;
                c->recs_in_pass[1] = prm.grouped_hist ? 0ull : n;
                Bucket b;
                b.offs = 0;
                b.count = static_cast<uint32_t>(n);
                b.first_tile = 0;
                b.ntiles = T1;
                b.src = SRC_IN;
                b.skip = 0;
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
}

// Array-of-structs records: decomposition into a key array and a value array,
// and the recomposition after the sort, one pass each at memory bandwidth.  A record is
// RW 4-byte words (key_bytes + value_bytes, the key at word KO); the key goes through the
// order-preserving bijection of its kind on the way in and back on the way out
// (P:907-918), fused into these passes.  Value words travel as opaque u32 / u64.
template <typename K>
__device__ __forceinline__ K key_map(K x, int kind, bool inv) {
    constexpr K SIGN = K(1) << (8 * sizeof(K) - 1);
    if (kind == 1) return x ^ SIGN;
    if (kind == 2) return !inv ? ((x & SIGN) ? ~x : (x ^ SIGN)) : ((x & SIGN) ? (x ^ SIGN) : ~x);
    return x;
}
template <typename K, typename V, int RW, bool KEYFIRST>
__global__ void k_records(const uint32_t *__restrict__ rec_in, uint32_t *__restrict__ rec_out, K *keys,
                          ValT<V> *vals, uint64_t n, int kind, int recompose) {
    pdl_wait();
    constexpr int KW = sizeof(K) / 4;
    constexpr int VW = HasVal<V>::value ? static_cast<int>(sizeof(ValT<V>)) / 4 : 0;
    constexpr int ko = KEYFIRST ? 0 : VW;  // word offset of the key
    static_assert(KW + VW == RW, "record = key + value words");
    const uint64_t stride = static_cast<uint64_t>(gridDim.x) * blockDim.x;
    for (uint64_t i = static_cast<uint64_t>(blockIdx.x) * blockDim.x + threadIdx.x; i < n; i += stride) {
        if (!recompose) {
            uint32_t w[RW];
#pragma unroll
            for (int j = 0; j < RW; ++j) w[j] = rec_in[i * RW + j];
            K k = 0;
#pragma unroll
            for (int j = 0; j < KW; ++j) k |= static_cast<K>(w[ko + j]) << (32 * j);
            keys[i] = key_map(k, kind, false);
            if constexpr (VW > 0) {
                ValT<V> v = 0;
                int q = 0;
#pragma unroll
                for (int j = 0; j < RW; ++j)
                    if (j < ko || j >= ko + KW) v |= static_cast<ValT<V>>(w[j]) << (32 * q++);
                vals[i] = v;
            }
        } else {
            const K k = key_map(keys[i], kind, true);
            uint32_t w[RW];
#pragma unroll
            for (int j = 0; j < KW; ++j) w[ko + j] = static_cast<uint32_t>(k >> (32 * j));
            if constexpr (VW > 0) {
                const ValT<V> v = vals[i];
                int q = 0;
#pragma unroll
                for (int j = 0; j < RW; ++j)
                    if (j < ko || j >= ko + KW) w[j] = static_cast<uint32_t>(v >> (32 * q++));
            }
#pragma unroll
            for (int j = 0; j < RW; ++j) rec_out[i * RW + j] = w[j];
        }
    }
}

template <typename T>
__global__ void k_copy(const T *__restrict__ in, T *__restrict__ out, uint64_t n) {
    const uint64_t stride = static_cast<uint64_t>(gridDim.x) * blockDim.x;
    for (uint64_t i = static_cast<uint64_t>(blockIdx.x) * blockDim.x + threadIdx.x; i < n; i += stride)
        out[i] = in[i];
}

// Copies of many pieces in one launch (the distributed sort's own pieces of the
// bucket-major exchange): the piece table travels in the kernel parameters (no host to
// device copy), {src_off, dst_off, count} in elements; the CTAs of the grid walk the
// pieces, each piece cut into chunks of CHUNK elements, 16-byte vectors where src and dst
// are equally aligned.
constexpr int COPY_PIECES_MAX = 256;
struct CopyPieces {
    uint64_t tab[3 * COPY_PIECES_MAX];
    uint32_t npieces;
};
template <typename T>
__global__ void __launch_bounds__(256) k_copy_pieces(const T *__restrict__ src, T *__restrict__ dst,
                                                     const __grid_constant__ CopyPieces prm) {
    pdl_wait();
    constexpr uint64_t CHUNK = 1u << 16;
    constexpr uint64_t VE = 16 / sizeof(T);
    for (uint32_t pc = 0; pc < prm.npieces; ++pc) {
        const uint64_t so = prm.tab[3 * pc], d = prm.tab[3 * pc + 1], cnt = prm.tab[3 * pc + 2];
        const uint64_t nch = (cnt + CHUNK - 1) / CHUNK;
        // chunk c of piece pc goes to CTA (pc + c) % grid: pieces are spread over the grid
        for (uint64_t c = (blockIdx.x + gridDim.x - pc % gridDim.x) % gridDim.x; c < nch; c += gridDim.x) {
            const uint64_t a = c * CHUNK, z = min(cnt, a + CHUNK);
            const T *sp = src + so;
            T *dp = dst + d;
            if (((so ^ d) % VE) == 0) {
                // scalar head to 16-byte alignment, vectors, scalar tail
                const uint64_t h = min(z, a + (VE - (so + a) % VE) % VE);
                for (uint64_t i = a + threadIdx.x; i < h; i += blockDim.x) dp[i] = sp[i];
                const uint64_t nv = (z - h) / VE;
                const uint4 *sv = reinterpret_cast<const uint4 *>(sp + h);
                uint4 *dv = reinterpret_cast<uint4 *>(dp + h);
                for (uint64_t v = threadIdx.x; v < nv; v += blockDim.x) dv[v] = sv[v];
                for (uint64_t i = h + nv * VE + threadIdx.x; i < z; i += blockDim.x) dp[i] = sp[i];
            } else {
                for (uint64_t i = a + threadIdx.x; i < z; i += blockDim.x) dp[i] = sp[i];
            }
        }
    }
}

// Sets the values of conditional graph nodes from the control block (small sorts replayed as
// a CUDA graph): what[i] = c < 8: local class list c is non-empty; 8: the counting local
// sort's hand-off list; 16 + c: the wide list of configuration c.
constexpr int MAX_CONDS = 16;
struct CondSet {
    cudaGraphConditionalHandle h[MAX_CONDS];
    uint32_t what[MAX_CONDS];
    int n;
    const Ctl *ctl;
};
static __global__ void k_set_conds(const __grid_constant__ CondSet cs) {
    pdl_wait();
    const int i = threadIdx.x;
    if (i < cs.n) {
        const uint32_t w = cs.what[i];
        const uint32_t v = w < 8 ? cs.ctl->nlocal[w] : (w == 8 ? cs.ctl->nlocal_fb2 : cs.ctl->nlocal_wide[w - 16]);
        cudaGraphSetConditional(cs.h[i], v != 0u ? 1u : 0u);
    }
}

static __global__ void k_fill_u64(uint64_t *p, uint64_t n, uint64_t v) {
    for (uint64_t i = static_cast<uint64_t>(blockIdx.x) * blockDim.x + threadIdx.x; i < n;
         i += static_cast<uint64_t>(gridDim.x) * blockDim.x)
        p[i] = v;
}

// ------------------------------------------------------------------ histogram

struct HistParams {
    const void *src_keys[3];  // indexed by SrcCode: each bucket's keys are in its src buffer
    uint64_t n;               // elements of the buffers
    int p;
    int lo;
    uint32_t mask;
    uint32_t kpb;
    const Bucket *buckets;
    uint32_t *tot;             // [bucket][256] of this pass (zeroed by the creator of the bucket)
    uint32_t *seg_last;        // [cta][256]: counts of the CTA's last bucket segment
    RangeMeta *seg_meta;       // [cta]
    TileDesc *tiles;           // [tile]: descriptor for k_scatter
    uint32_t *tile_pref;       // [tile][256]: digit counts of the earlier tiles of its bucket segment
    Ctl *ctl;
    int kind;  // hrs_key_kind: keys still in the input go through the bijection
};

// One CTA walks a contiguous run of tiles [tb, te) (the same runs as k_scatter): per tile a
// block histogram of the digit (plain shared atomics: on B200 they run at the same rate for
// any skew, profiles/r01_micro_hist.txt), the tile's prefix within its bucket segment and
// its descriptor for the scatter.  The keys come straight from global memory in 16-byte
// vectors (no staging: every resident CTA keeps a whole tile of loads in flight), and one
// barrier per tile suffices: the histograms and the tile records are double-buffered, the
// counts of tile i are folded in after the barrier that ends its counting.
#ifndef HRS_HIST_MINB
#define HRS_HIST_MINB 4
#endif
#ifndef HRS_HIST_PF
#define HRS_HIST_PF 1
#endif
// element q of a 16-byte vector of keys (no address taken: the vector stays in registers)
template <typename K>
__device__ __forceinline__ K vec_elem(const uint4 &v, int q) {
    if constexpr (sizeof(K) == 4) return static_cast<K>(q == 0 ? v.x : q == 1 ? v.y : q == 2 ? v.z : v.w);
    else return static_cast<K>(q == 0 ? (static_cast<unsigned long long>(v.y) << 32 | v.x)
                                      : (static_cast<unsigned long long>(v.w) << 32 | v.z));
}
struct HistTile {
    uint64_t offs;
    uint32_t count, bucket, flush, src;
};

template <typename K, int THREADS, int CAP, bool TY>
__global__ void __launch_bounds__(THREADS, HRS_HIST_MINB) k_hist(HistParams prm) {
    pdl_wait();
    static_assert(THREADS >= RADIX, "one thread per digit for the tile prefixes");
    constexpr int VK = 16 / sizeof(K);
    constexpr int NV = (CAP / VK + THREADS - 1) / THREADS;  // whole vectors of a tile per thread
    // HRS_HIST_PF: the loads of tile t + 1 are issued as soon as tile t's keys are counted,
    // before the barrier that ends tile t (its descriptor was published a tile earlier:
    // three descriptor slots), so they overlap the barrier and the fold
    constexpr int NTI = HRS_HIST_PF ? 3 : 2;
    __shared__ uint32_t wh[2][RADIX];
    __shared__ HistTile ti[NTI];
    __shared__ TileCursor cur;
    const int tid = threadIdx.x;
    const unsigned long long al = prm.ctl->alloc[prm.p];
    const uint32_t T = alloc_tiles(al), NB = alloc_buckets(al);
    const uint32_t tb = range_begin(T, blockIdx.x, gridDim.x), te = range_begin(T, blockIdx.x + 1, gridDim.x);
    if (tb >= te) {
        if (tid == 0) prm.seg_meta[blockIdx.x] = RangeMeta{EMPTY_RANGE, EMPTY_RANGE};
        return;
    }
    auto publish = [&](int slot) {  // tid 0: the cursor's tile into ti[slot], then advance
        HistTile h;
        h.offs = cur.offs();
        h.count = cur.count();
        h.bucket = cur.b;
        h.flush = cur.last_of_bucket() || cur.t + 1 == te;
        h.src = cur.bk.src;
        ti[slot] = h;
        cur.next();
    };
    if (tid == 0) {
        cur.start(prm.buckets, NB, tb, te, prm.kpb);
        prm.seg_meta[blockIdx.x].first_bucket = cur.b;
        publish(0);
        if (HRS_HIST_PF && tb + 1 < te) publish(1);
    }
    for (int i = tid; i < 2 * RADIX; i += THREADS) (&wh[0][0])[i] = 0;
    __syncthreads();
    // a tile's key vectors: [0, h0) before the first 16-byte boundary, nvec whole vectors,
    // the tail after them (edge elements: ne < 2 VK, one per thread)
    struct Geo {
        const K *src;
        uint32_t h0, nvec, tail0, ne;
        bool mapin;
    };
    auto geo = [&](const HistTile &in) {
        Geo g;
        // (selected, not indexed: a dynamic index would copy the parameters to local memory)
        const void *kb = in.src == SRC_IN ? prm.src_keys[SRC_IN] : in.src == SRC_AUX ? prm.src_keys[SRC_AUX] : prm.src_keys[SRC_OUT];
        g.src = static_cast<const K *>(kb) + in.offs;
        g.mapin = TY && prm.kind != 0 && in.src == SRC_IN;
        const uint32_t mis = static_cast<uint32_t>(reinterpret_cast<uintptr_t>(g.src) / sizeof(K)) % VK;
        g.h0 = min(in.count, (VK - mis) % VK);
        g.nvec = (in.count - g.h0) / VK;
        g.tail0 = g.h0 + g.nvec * VK;
        g.ne = g.h0 + (in.count - g.tail0);
        return g;
    };
    uint4 w[NV];
    K ek = K(0);
    auto load = [&](const Geo &g) {
        const uint4 *vp = reinterpret_cast<const uint4 *>(g.src + g.h0);
#pragma unroll
        for (int j = 0; j < NV; ++j) {
            const uint32_t v = tid + j * THREADS;
            if (v < g.nvec) w[j] = __ldcs(vp + v);
        }
        if (static_cast<uint32_t>(tid) < g.ne) ek = g.src[static_cast<uint32_t>(tid) < g.h0 ? tid : g.tail0 + (tid - g.h0)];
    };
    if constexpr (HRS_HIST_PF) load(geo(ti[0]));
    uint32_t seg_run = 0;   // digit tid: count of the current bucket segment before this tile
    bool first_seg = true;  // inside the CTA's first bucket segment (its carry applies)
    for (uint32_t t = tb, it = 0; t < te; ++t, ++it) {
        const HistTile in = ti[it % NTI];
        const Geo g = geo(in);
        if constexpr (!HRS_HIST_PF) load(g);
        if (tid == 0 && t + (NTI - 1) < te) publish((it + NTI - 1) % NTI);
        // tile descriptor and tile-ordered prefix for the scatter
        if (tid < RADIX) prm.tile_pref[static_cast<uint64_t>(t) * RADIX + tid] = seg_run;
        if (tid == 0) {
            TileDesc td;
            td.offs = in.offs;
            td.count = in.count;
            td.bucket = in.bucket;
            td.carry_row = first_seg ? blockIdx.x : EMPTY_RANGE;
            td.pad = 0;
            prm.tiles[t] = td;
        }
        uint32_t *my = wh[it & 1u];
        auto dig = [&](K k) { return digit_of(g.mapin ? key_map(k, prm.kind, false) : k, prm.lo, prm.mask); };
#pragma unroll
        for (int j = 0; j < NV; ++j) {
            if (tid + j * THREADS < g.nvec) {
#pragma unroll
                for (int q = 0; q < VK; ++q) atomicAdd(&my[dig(vec_elem<K>(w[j], q))], 1u);
            }
        }
        if (static_cast<uint32_t>(tid) < g.ne) atomicAdd(&my[dig(ek)], 1u);
        // (PF: ti[(it + 1) % 3] was published before the previous barrier)
        if (HRS_HIST_PF && t + 1 < te) load(geo(ti[(it + 1) % NTI]));
        __syncthreads();  // the tile's counts are complete; the next descriptor is published
        if (tid < RADIX) {
            seg_run += my[tid];
            my[tid] = 0;  // (counted into again two tiles on, after the next barrier)
        }
        if (in.flush) {
            const bool last_seg = t + 1 == te;
            if (tid < RADIX) {
                if (seg_run) atomicAdd(&prm.tot[static_cast<uint64_t>(in.bucket) * RADIX + tid], seg_run);
                if (last_seg) prm.seg_last[static_cast<uint64_t>(blockIdx.x) * RADIX + tid] = seg_run;
            }
            if (last_seg && tid == 0) prm.seg_meta[blockIdx.x].last_bucket = in.bucket;
            seg_run = 0;
            first_seg = false;
        }
    }
}

// ------------------------------------------------------------------ classification (one CTA per bucket)

struct ClassifyParams {
    int p;
    int last;  // 1: digit p is the least-significant one (no further classification)
    int lo;    // digit bits [lo, lo + width)
    int width;
    Bucket *buckets;  // (k_classify sets Bucket::skip)
    const uint32_t *tot;  // this pass
    uint32_t *tot_next;   // next pass (rows of created buckets are cleared)
    Bucket *next_buckets;
    uint32_t *sub_rel;  // [bucket][256] sub-bucket starts relative to the bucket
    const uint32_t *seg_last;
    const RangeMeta *seg_meta;
    uint32_t *carry;    // [cta][256]: tiles of the CTA's first bucket before its range
    uint32_t ranges;    // CTAs of the hist/scatter grid
    Ctl *ctl;
    LocalEntry *local[HRS_NUM_CLASSES];
    uint32_t local_cap[HRS_NUM_CLASSES];
    uint32_t tile_cap, bucket_cap;
    uint32_t lt, mt, kpb;
    int single_class;       // >= 0: every local entry goes to this class (ablation)
    uint16_t src_code;      // buffer holding X_p
    uint64_t *out_hist;     // building block: the root bucket's histogram
    uint64_t *out_offsets;  // building block: the root bucket's sub-bucket starts (+ n)
};

// Block-wide suffix minimum of one value per thread (THREADS == 256 = RADIX threads,
// thread d holds digit d): returns min(v[d .. 255]).  wbuf: 8 words.
__device__ __forceinline__ uint32_t block_suffix_min256(uint32_t v, uint32_t *wbuf) {
    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
        const uint32_t y = __shfl_down_sync(0xffffffffu, v, o);
        if (lane + o < 32) v = min(v, y);
    }
    if (lane == 0) wbuf[warp] = v;  // the minimum of the warp's 32 digits
    __syncthreads();
#pragma unroll
    for (int w = 0; w < RADIX / 32; ++w) v = w > warp ? min(v, wbuf[w]) : v;
    __syncthreads();  // wbuf is reused by the next call
    return v;
}

// The greedy merge of the local candidates of one bucket (reading #5 of DESIGN.md: in
// digit order, a candidate joins the open group while the group stays below ∂, a
// sibling > ∂ˆ closes it, empty sub-buckets are skipped), computed by one thread per
// digit instead of one thread walking 256 digits.  With P = exclusive prefix of the
// sub-bucket sizes, the group that starts at candidate i ends at
//     gend(i) = min(first sibling > ∂ˆ after i,  first k > i with P[k+1] >= P[i] + ∂)
// (it holds the candidates of [i, gend), size P[gend] - P[i]) and the next group
// starts at the first candidate >= gend.  The groups are the chain of starts from the
// first candidate, marked by pointer doubling (8 rounds for 256 digits).
// Writes glead[i] = group size and gmulti[i] = (>= 2 members ? group end : 0) at every
// group start i.
template <int THREADS>
__device__ void merge_groups(const ClassifyParams &prm, const uint32_t *tot, const uint32_t *P, uint32_t *glead,
                             uint32_t *gmulti, uint32_t *ws) {
    static_assert(THREADS == RADIX, "one thread per digit");
    uint32_t *jmp = ws;               // [2][NBINS] successor tables (double-buffered)
    uint32_t *flag = ws + 2 * NBINS;  // [NBINS] group start
    uint32_t *wbuf = ws + 3 * NBINS;  // [8]
    const uint32_t d = threadIdx.x;
    const uint32_t s = tot[d];
    const bool cand = s > 0 && s <= prm.lt, big = s > prm.lt;
    // first big sibling after d, first candidate at or after d (256 = none)
    const uint32_t nb_incl = block_suffix_min256(big ? d : RADIX, wbuf);
    const uint32_t nc = block_suffix_min256(cand ? d : RADIX, wbuf);
    flag[d] = nc;  // (temporary: NC table, read below)
    jmp[d] = nb_incl;
    if (d == 0) {
        flag[RADIX] = RADIX;
        jmp[RADIX] = RADIX;
    }
    __syncthreads();
    uint32_t succ = RADIX, gend = RADIX, size = 0;
    bool multi = false;
    if (cand) {
        const uint32_t b = jmp[d + 1];  // first big after d
        // first q in [d + 2, 256] with P[q] >= P[d] + ∂ (k = q - 1), else k = 256
        const uint32_t target = P[d] + prm.mt;
        uint32_t lo = d + 2, hi = RADIX + 1;  // answer in [lo, hi); hi = none
        while (lo < hi) {
            const uint32_t mid = (lo + hi) >> 1;
            if (P[mid] >= target) hi = mid;
            else lo = mid + 1;
        }
        const uint32_t k1 = lo <= RADIX ? lo - 1 : RADIX;
        gend = min(k1, b);
        size = P[gend] - P[d];
        succ = flag[gend];           // first candidate >= gend
        multi = flag[d + 1] < gend;  // a second candidate inside the group
    }
    const uint32_t first = flag[0];
    __syncthreads();  // NC / NB tables consumed
    jmp[d] = succ;
    flag[d] = d == first ? 1u : 0u;
    if (d == 0) jmp[RADIX] = RADIX;
    __syncthreads();
    uint32_t *ja = jmp, *jb = jmp + NBINS;
    for (int round = 0; round < 8; ++round) {
        const uint32_t j = ja[d];
        if (flag[d] && j < RADIX) flag[j] = 1u;  // (flags only ever go 0 -> 1)
        jb[d] = j < RADIX ? ja[j] : RADIX;
        if (d == 0) jb[RADIX] = RADIX;
        __syncthreads();
        uint32_t *t = ja;
        ja = jb;
        jb = t;
    }
    if (cand && flag[d]) {
        glead[d] = size;
        gmulti[d] = multi ? gend : 0u;  // (> d: the group's digits are [d, gend))
    }
}

template <int THREADS>
__device__ void classify_bucket(const ClassifyParams &prm, const Bucket &bk, uint32_t bucket_id, uint32_t *sm) {
    static_assert(THREADS >= RADIX, "one thread per digit");
    uint32_t *tot = sm;                 // 256 (+1)
    uint32_t *start = sm + 1 * NBINS;   // exclusive prefix of tot
    uint32_t *ct = sm + 2 * NBINS;      // child tiles per digit -> exclusive
    uint32_t *cb = sm + 3 * NBINS;      // child flag per digit -> exclusive
    uint32_t *glead = sm + 4 * NBINS;   // local group size at the leader digit (0 = none)
    uint32_t *gmulti = sm + 5 * NBINS;  // group end if the group merged >= 2 sub-buckets, else 0
    uint32_t *misc = sm + 6 * NBINS;    // [0] base tile, [1] base bucket, [2..9] class counts, [10..17] class bases
    const int tid = threadIdx.x;
    for (int d = tid; d < NBINS; d += THREADS) {
        const uint32_t v = d < RADIX ? prm.tot[static_cast<uint64_t>(bucket_id) * RADIX + d] : 0u;
        tot[d] = v;
        start[d] = v;
        glead[d] = 0;
        gmulti[d] = 0;
        const bool cnt = !prm.last && v > prm.lt;
        ct[d] = cnt ? v / prm.kpb + (v % prm.kpb != 0u) : 0u;  // (no u32 wrap near 2^32)
        cb[d] = cnt ? 1u : 0u;
    }
    if (tid < 32) misc[tid] = 0;
    __syncthreads();
    warp0_exclusive_scan(start, NBINS);
    __syncthreads();
    warp0_exclusive_scan(ct, NBINS);
    __syncthreads();
    warp0_exclusive_scan(cb, NBINS);
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

    // ---- a bucket that never moved (still in the input) whose digit p is the same for all
    // of its records keeps its records where they are: the scatter of pass p would only copy
    // it (reading #22); its child and local entries point at the input
    const bool skip = __syncthreads_or(tid < RADIX && tot[tid] == bk.count) && bk.src == SRC_IN;
    const uint16_t child_src = skip ? static_cast<uint16_t>(SRC_IN) : prm.src_code;
    if (skip && tid == 0) {
        prm.buckets[bucket_id].skip = 1;
        atomicAdd(&prm.ctl->skipped_in_pass[prm.p], static_cast<unsigned long long>(bk.count));
    }

    // ---- counting children: next-pass buckets (R2) and their tile ranges (R4); one
    // 64-bit atomic allocates both so bucket order stays tile order
    const uint32_t TT = ct[RADIX];
    const uint32_t NC = cb[RADIX];
    if (tid == 0) {
        uint32_t bt = 0, bb = 0;
        if (NC) {
            const unsigned long long a = atomicAdd(&prm.ctl->alloc[prm.p + 1],
                                                   (static_cast<unsigned long long>(TT) << 32) | NC);
            bt = alloc_tiles(a);
            bb = alloc_buckets(a);
            if (static_cast<uint64_t>(bt) + TT > prm.tile_cap || static_cast<uint64_t>(bb) + NC > prm.bucket_cap)
                atomicExch(&prm.ctl->overflow, 1u);
        }
        misc[0] = bt;
        misc[1] = bb;
    }
    // ---- local candidates: greedy merge (R3 / reading #5)
    bool has_small = false;
    for (int d = tid; d < RADIX; d += THREADS) {
        const uint32_t s = tot[d];
        if (s > 0 && s <= prm.lt && s < prm.mt) has_small = true;
    }
    has_small = __syncthreads_or(has_small);
    if (!has_small) {
        // no sub-bucket can merge: every candidate is its own group
        for (int d = tid; d < RADIX; d += THREADS) {
            const uint32_t s = tot[d];
            if (s > 0 && s <= prm.lt) glead[d] = s;
        }
    } else {
        merge_groups<THREADS>(prm, tot, start, glead, gmulti, sm + 7 * NBINS);
    }
    __syncthreads();
    // per-class slot allocation
    int my_cls = -1;
    uint32_t my_slot = 0;
    if (tid < RADIX && glead[tid]) {
        my_cls = prm.single_class >= 0 ? prm.single_class : size_class_of(glead[tid]);
        my_slot = atomicAdd(&misc[2 + my_cls], 1u);
    }
    // statistics: warp reductions of the next pass's records, local records, merged groups
    unsigned long long recs_next = 0, lrecs = 0, merged = 0;
    if (tid < RADIX) {
        const uint32_t s = tot[tid];
        if (s > prm.lt) recs_next = s;
        lrecs = glead[tid];
        merged = gmulti[tid] ? 1u : 0u;
    }
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) {
        recs_next += __shfl_xor_sync(0xffffffffu, recs_next, o);
        lrecs += __shfl_xor_sync(0xffffffffu, lrecs, o);
        merged += __shfl_xor_sync(0xffffffffu, merged, o);
    }
    if ((tid & 31) == 0 && tid < RADIX) {
        if (recs_next) atomicAdd(&prm.ctl->recs_in_pass[prm.p + 1], recs_next);
        if (lrecs) atomicAdd(&prm.ctl->local_recs, lrecs);
        if (merged) atomicAdd(&prm.ctl->merged_groups, merged);
    }
    __syncthreads();
    if (tid < HRS_NUM_CLASSES) {
        const uint32_t cnt = misc[2 + tid];
        const uint32_t base = cnt ? atomicAdd(&prm.ctl->nlocal[tid], cnt) : 0u;
        if (cnt && base + cnt > prm.local_cap[tid]) atomicExch(&prm.ctl->overflow, 1u);
        misc[10 + tid] = base;
    }
    __syncthreads();
    if (my_cls >= 0) {
        const uint32_t slot = misc[10 + my_cls] + my_slot;
        if (slot < prm.local_cap[my_cls]) {
            LocalEntry e;
            e.offs = boffs + start[tid];
            e.count = glead[tid];
            // a merged group sorts the digit bits in which its members differ (reading #6: the
            // bits of [hi_bit, hi_p) are common to digits tid .. last): the local sort's
            // counted bits start at its top varying bit
            int hb = prm.lo;
            if (gmulti[tid]) {
                uint32_t last = gmulti[tid] - 1u;
                while (last > static_cast<uint32_t>(tid) && tot[last] == 0u) --last;  // last non-empty member
                hb = prm.lo + (32 - __clz(static_cast<int>(static_cast<uint32_t>(tid) ^ last)));
            }
            e.hi_bit = static_cast<uint16_t>(hb);
            e.src = child_src;
            prm.local[my_cls][slot] = e;
        }
    }
    // child buckets (their histogram rows of the next pass are cleared here)
    const uint32_t bt = misc[0], bb = misc[1];
    if (tid < RADIX) {
        const uint32_t s = tot[tid];
        const uint32_t id = bb + cb[tid];
        if (s > prm.lt && id < prm.bucket_cap) {
            Bucket nb;
            nb.offs = boffs + start[tid];
            nb.count = s;
            nb.first_tile = bt + ct[tid];
            nb.ntiles = s / prm.kpb + (s % prm.kpb != 0u);
            nb.src = child_src;
            nb.skip = 0;
            prm.next_buckets[id] = nb;
        }
    }
    for (uint32_t i = tid; i < NC * RADIX; i += THREADS) {
        const uint32_t id = bb + i / RADIX;
        if (id < prm.bucket_cap) prm.tot_next[static_cast<uint64_t>(id) * RADIX + (i % RADIX)] = 0;
    }
}

// Carry of every hist/scatter CTA: the digit counts of the tiles of its first bucket
// that precede its range (an exclusive scan over CTAs, segmented by bucket).  One
// thread per digit walks the CTAs; the loads are batched so their latencies overlap.
// The carry of every CTA range (the digit counts of the tiles of its first bucket that lie
// in earlier ranges): a scan over the ranges, segmented where a bucket ends, one per digit.
// CARRY_CTAS blocks split the digits; inside a block the ranges are cut into
// THREADS / (RADIX / CARRY_CTAS) chunks scanned in parallel: first each chunk's outgoing run
// assuming none comes in (and whether an incoming run would flow through it), then the runs
// entering the chunks in chunk order, then each chunk's scan again from its true incoming
// run, writing the carries.
#ifndef HRS_CARRY_CTAS
#define HRS_CARRY_CTAS 32  // measured: 8 -> 32 CTAs, c2 classify 0.019 + 0.019 -> 0.013 + 0.011 ms (64: 0.013 + 0.015)
#endif
constexpr int CARRY_CTAS = HRS_CARRY_CTAS;
template <int THREADS>
__device__ void range_carries(const ClassifyParams &prm, uint32_t part) {
    constexpr int DPB = RADIX / CARRY_CTAS;  // digits per block
    constexpr int NQ = THREADS / DPB;        // chunks of ranges
    constexpr int B = 32;
    static_assert(THREADS % DPB == 0 && NQ >= 1, "carry geometry");
    __shared__ uint32_t out_run[NQ][DPB], out_pass[NQ][DPB];
    const RangeMeta *__restrict__ meta = prm.seg_meta;
    const uint32_t *__restrict__ segl = prm.seg_last;
    uint32_t *__restrict__ carry = prm.carry;
    const uint32_t dl = threadIdx.x % DPB, d = part * DPB + dl, q = threadIdx.x / DPB;
    const uint32_t R = prm.ranges;
    const uint32_t c0 = static_cast<uint32_t>((static_cast<uint64_t>(R) * q) / NQ);
    const uint32_t c1 = static_cast<uint32_t>((static_cast<uint64_t>(R) * (q + 1)) / NQ);
    uint32_t last0 = EMPTY_RANGE;  // last bucket of the last non-empty range before c0
    for (uint32_t c = c0; c-- > 0;) {
        const RangeMeta m = meta[c];
        if (m.first_bucket != EMPTY_RANGE) {
            last0 = m.last_bucket;
            break;
        }
    }
    // scan of the chunk from run `in`; WRITE: store the carries
    auto scan = [&](uint32_t in, bool write, bool &pass) -> uint32_t {
        uint32_t run = in, prev_last = last0;
        pass = true;
        for (uint32_t cb = c0; cb < c1; cb += B) {
            RangeMeta m[B];
            uint32_t sl[B];
#pragma unroll
            for (int i = 0; i < B; ++i) {
                if (cb + i < c1) {
                    m[i] = meta[cb + i];
                    sl[i] = segl[static_cast<uint64_t>(cb + i) * RADIX + d];
                } else {
                    m[i].first_bucket = EMPTY_RANGE;
                    m[i].last_bucket = EMPTY_RANGE;
                    sl[i] = 0;
                }
            }
#pragma unroll
            for (int i = 0; i < B; ++i) {
                if (m[i].first_bucket == EMPTY_RANGE) continue;
                const bool cont = m[i].first_bucket == prev_last;
                const uint32_t car = cont ? run : 0u;
                if (write) carry[static_cast<uint64_t>(cb + i) * RADIX + d] = car;
                pass = pass && cont && m[i].first_bucket == m[i].last_bucket;
                run = (m[i].first_bucket == m[i].last_bucket) ? car + sl[i] : sl[i];
                prev_last = m[i].last_bucket;
            }
        }
        return run;
    };
    bool pass;
    uint32_t inc = 0;  // the run entering chunk q
    if (NQ > 1) {
        out_run[q][dl] = scan(0u, false, pass);
        out_pass[q][dl] = pass;
        __syncthreads();
        for (uint32_t r = 0; r < q; ++r) inc = out_run[r][dl] + (out_pass[r][dl] ? inc : 0u);
    }
    scan(inc, true, pass);
}

template <int THREADS>
__global__ void __launch_bounds__(THREADS) k_classify(ClassifyParams prm) {
    pdl_wait();
    __shared__ uint32_t scratch[11 * NBINS];  // classify_bucket: 7 rows, merge_groups: 3 rows + 8 words
    const uint32_t nb = alloc_buckets(prm.ctl->alloc[prm.p]);
    if (nb == 0) return;  // nothing reached this pass
    // the last CARRY_CTAS blocks compute the range carries, the others classify buckets
    const uint32_t nblk = gridDim.x - CARRY_CTAS;
    if (blockIdx.x >= nblk) {
        range_carries<THREADS>(prm, blockIdx.x - nblk);
        return;
    }
    for (uint32_t b = blockIdx.x; b < nb; b += nblk) {
        const Bucket bk = prm.buckets[b];
        classify_bucket<THREADS>(prm, bk, b, scratch);
        __syncthreads();
    }
}

// ------------------------------------------------------------------ scatter

struct ScatterParams {
    uint64_t n;  // elements of the buffers
    const void *src_keys[3];  // indexed by SrcCode (Bucket::src): where each bucket's records are
    void *keys_out;           // X_p
    const void *src_vals[3];
    void *vals_out;
    int p;
    int lo;
    uint32_t mask;
    const Bucket *buckets;
    const uint32_t *sub_rel;
    const uint32_t *carry;
    const TileDesc *tiles;
    const uint32_t *tile_pref;
    Ctl *ctl;
    int force_redo;  // HRS_FLAG_FORCE_REDO: every stability check fails (tests of the redo path)
    int kind;        // hrs_key_kind: the bijection on the way out of the input, its inverse
    int final_pass;  //   on the way into the final output (the last pass)
    // small sorts replayed as a CUDA graph: the next pass is a conditional node whose value
    // this scatter sets (the next pass has buckets), so empty passes cost nothing
    cudaGraphConditionalHandle next_cond;
    int has_next_cond;
    // DST instantiation (hrs_partition_pass_to, the fused exchange of SURVEY §8(f) N2): digit
    // d's run goes to window w = dst_off[d] >> 48 at element offset dst_off[d] & (2^48 - 1);
    // window w is the device address of a key (value) array, possibly another GPU's memory
    // mapped over NVLink
    const unsigned long long *dst_off;    // [2^width]
    const unsigned long long *dst_kwin;   // [windows]
    const unsigned long long *dst_vwin;   // [windows]
};
constexpr unsigned long long DST_OFF_MASK = (1ull << 48) - 1;

struct StageInfo {
    uint32_t valid, count, bucket, carry_row, kpad, k0, k1, vpad, v0, v1, tile, src;
    uint64_t offs;
};

// Shared memory of one scatter CTA (NBUF staging buffers of keys and values, filled by
// TMA bulk copies).  The rank needs per-warp digit counters [W][256] and the tile's digit
// starts; the sorted tile is built IN PLACE in the key staging buffer (the keys are held
// in registers from the count on) plus a 16-bit slot -> element index (sidx) through which
// the values are gathered and the stability of the fast rank is checked.
template <typename K, typename V, int THREADS, int KPT, int NBUF, bool DST = false>
struct ScatterSmem {
    static constexpr int W = THREADS / 32;
    static constexpr int KPB = THREADS * KPT;
    using VT = ValT<V>;
    static constexpr bool HV = HasVal<V>::value;
    static constexpr size_t kst_elems = KPB + 32 / sizeof(K);
    static constexpr size_t vst_elems = KPB + 32 / sizeof(VT);
    // VS: the values are staged in ONE buffer (own barrier), loaded after the previous
    // tile's write-out, while the keys keep two: the freed buffer buys a larger tile
    static constexpr bool VS = HRS_SC_VSPLIT && !HRS_SC_DIRECT && NBUF == 2 && HV;
    static constexpr size_t off_bar = 0;  // [3]: key stages, value stage
    static constexpr size_t off_vinfo = 24;
    static constexpr size_t off_info = 48;
    static constexpr size_t off_cnt = align16(off_info + NBUF * sizeof(StageInfo));
    static constexpr size_t off_wsum = align16(off_cnt + sizeof(uint32_t) * W * RADIX);
    static constexpr size_t off_gs = align16(off_wsum + sizeof(uint32_t) * 16);
    // PTR (8-byte keys and values): gs holds 16 bytes per digit -- the address of slot 0's
    // destination and the first slot -- so a write-out address is one add (measured: c4
    // scatter 3.94 -> 3.71 ms; with 4-byte records the wider lookup costs more shared-memory
    // wavefronts than the address arithmetic it saves, measured slower)
    static constexpr bool PTR = !DST && !HRS_SC_DIRECT && sizeof(K) == 8 && (!HV || sizeof(VT) == 8);
    static constexpr size_t off_start = align16(off_gs + (PTR ? sizeof(uint4) : sizeof(uint2)) * RADIX);  // DST: digit starts
    static constexpr size_t off_sidx = align16(off_start + (DST ? sizeof(uint32_t) * RADIX : 0));
    static constexpr size_t off_kst = align16(off_sidx + sizeof(uint16_t) * KPB);
    static constexpr size_t kst_bytes = align16(sizeof(K) * kst_elems);
    static constexpr size_t off_vst = off_kst + NBUF * kst_bytes;
    static constexpr size_t vst_bytes = HV ? align16(sizeof(VT) * vst_elems) : 0;
    static constexpr size_t bytes = off_vst + (VS ? 1 : NBUF) * vst_bytes;
};

// One counting pass over the tiles of every bucket of pass p, stable.
// Per tile, with the next tile already in flight through TMA (NBUF = 2) or the other
// resident CTAs covering the load (NBUF = 1):
//   A  count: every warp ranks its 32 x KPT keys (warp-striped, element e = warp*32*KPT +
//      c*32 + lane) against its own digit counters: the returning atomic of the fast rank
//      gives the in-warp rank (lane order of same-address lanes, checked below), the exact
//      rank (skewed tiles) counts each column and orders duplicates with one match-any;
//   B  fold: thread d sums the W warp counters of digit d, a block scan of the digit
//      totals gives the tile's digit starts, and every warp counter becomes the first slot
//      of that warp's run of digit d (one thread per digit, all counters touched once);
//   C  place: slot = counter + in-warp rank; the key (held in a register) is stored at its
//      slot in the key staging buffer, the element index in sidx;
//   D  write-out: slot j holds key ks[j] and value vs[sidx[j]], destination = global base
//      of digit d + j - start[d]: consecutive threads store consecutive addresses of every
//      digit run (write-combined, Fig 3).  Slot j - 1 of the same digit must
//      hold an earlier element -- the complete stability condition; a tile that fails it
//      (or every tile under HRS_FLAG_FORCE_REDO) is ranked again with the exact rank.
// The per-digit global base of a tile (sub-bucket start + counts of the earlier tiles of
// its bucket) comes from k_hist / k_classify, so tiles are independent (no
// look-back) and claimed in order from a counter: the tiles in flight write neighbouring
// runs of every sub-bucket, which combine in L2.
template <typename K, typename V, int THREADS, int KPT, int MINB, int NBUF, bool TY, bool DST = false>
__global__ void __launch_bounds__(THREADS, MINB) k_scatter(ScatterParams prm) {
    pdl_wait();
    static_assert(NBUF == 1 || NBUF == 2, "one or two staging buffers");
    static_assert(THREADS % RADIX == 0 && THREADS <= 4 * RADIX, "threads 0..255 fold one digit each");
    static_assert(32 * KPT < (1 << 16), "the in-warp rank is packed above the digit");
    using L = ScatterSmem<K, V, THREADS, KPT, NBUF, DST>;
    constexpr bool VS = L::VS;
    static_assert(!DST || THREADS * KPT < (1 << 16), "DST packs a tile slot and a window into 32 bits");
    constexpr int W = THREADS / 32;
    constexpr bool HV = HasVal<V>::value;
    using VT = ValT<V>;
    extern __shared__ __align__(16) unsigned char smem[];
    uint64_t *bar = reinterpret_cast<uint64_t *>(smem + L::off_bar);
    StageInfo *info = reinterpret_cast<StageInfo *>(smem + L::off_info);
    Seg *vinfo = reinterpret_cast<Seg *>(smem + L::off_vinfo);  // VS: the value stage's segment
    uint32_t *cnt = reinterpret_cast<uint32_t *>(smem + L::off_cnt);    // [W][256]
    uint32_t *wsum = reinterpret_cast<uint32_t *>(smem + L::off_wsum);  // [W] digit-total partial sums
    // gs[d] = {destination of slot 0 of digit d relative to the bucket (may wrap), first slot of d}
    uint2 *gs = reinterpret_cast<uint2 *>(smem + L::off_gs);
    // DST: gs[d] = the 64-bit (window << 48 | element offset of slot 0 of digit d), sstart[d]
    uint32_t *sstart = reinterpret_cast<uint32_t *>(smem + L::off_start);
    uint16_t *sidx = reinterpret_cast<uint16_t *>(smem + L::off_sidx);
    auto kst = [&](int s) { return reinterpret_cast<K *>(smem + L::off_kst + s * L::kst_bytes); };
    auto vst = [&](int s) { return reinterpret_cast<VT *>(smem + L::off_vst + s * L::vst_bytes); };

    K *__restrict__ kout = static_cast<K *>(prm.keys_out);
    VT *__restrict__ vout = static_cast<VT *>(prm.vals_out);
    auto kin_of = [&](uint32_t src) { return static_cast<const K *>(prm.src_keys[src]); };
    auto vin_of = [&](uint32_t src) { return static_cast<const VT *>(prm.src_vals[src]); };
    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    const uint32_t wbase = static_cast<uint32_t>(warp) * 32 * KPT;
    const uint32_t T = alloc_tiles(prm.ctl->alloc[prm.p]);
    if (prm.has_next_cond && blockIdx.x == 0 && threadIdx.x == 0)  // (k_classify of this pass has completed)
        cudaGraphSetConditional(prm.next_cond, alloc_buckets(prm.ctl->alloc[prm.p + 1]) != 0u ? 1u : 0u);
    if (blockIdx.x >= T) return;
    const uint64_t pol = policy_evict_first();
    // HRS_SC_STHINT: the write-out's stores carry an L2 evict_last hint (1: first pass only,
    // whose write frontiers are spread over the whole output; 2: every pass)
    const bool sthint = HRS_SC_STHINT == 2 || (HRS_SC_STHINT == 1 && prm.p == 1);
    const uint64_t spol = HRS_SC_STHINT ? policy_evict_last() : 0ull;
    uint32_t *const ca = cnt + warp * RADIX;  // this warp's counters
    for (int i = tid; i < W * RADIX; i += THREADS) cnt[i] = 0;

    auto issue = [&](int s, uint32_t t) {
        StageInfo &in = info[s];
        TileDesc td;
        uint32_t src = SRC_IN;
        while (t < T) {  // (the tiles of a skipped bucket are passed over: the claim jumps past them)
            td = prm.tiles[t];
            const Bucket bk = prm.buckets[td.bucket];
            src = bk.src;
            if (!bk.skip) break;
            atomicMax(&prm.ctl->claim[prm.p], bk.first_tile + bk.ntiles);
            t = atomicAdd(&prm.ctl->claim[prm.p], 1u);
        }
        in.valid = t < T;
        if (t >= T) return;
        const K *kin = kin_of(src);
        const VT *vin = HV ? vin_of(src) : nullptr;
        in.src = src;
        in.count = td.count;
        in.bucket = td.bucket;
        in.carry_row = td.carry_row;
        in.offs = td.offs;
        in.tile = t;
        Seg sk, sv;
        uint32_t bytes = seg_plan(kin + td.offs, td.count, kin, kin + prm.n, sk);
        in.kpad = sk.pad;
        in.k0 = static_cast<uint32_t>(sk.i0);
        in.k1 = static_cast<uint32_t>(sk.i1);
        if (HV && !VS) {
            bytes += seg_plan(vin + td.offs, td.count, vin, vin + prm.n, sv);
            in.vpad = sv.pad;
            in.v0 = static_cast<uint32_t>(sv.i0);
            in.v1 = static_cast<uint32_t>(sv.i1);
        }
        mbar_arrive_expect_tx(&bar[s], bytes);
        seg_issue(kst(s), kin + td.offs, sk, &bar[s], pol);
        if (HV && !VS) seg_issue(vst(s), vin + td.offs, sv, &bar[s], pol);
    };
    // VS: the values of a tile whose keys are staged (the segment is published through
    // the barrier: written before the arrive, read after the wait)
    auto vissue = [&](const StageInfo &in) {
        if (!in.valid) return;
        const VT *vin = vin_of(in.src);
        Seg sv;
        const uint32_t bytes = seg_plan(vin + in.offs, in.count, vin, vin + prm.n, sv);
        *vinfo = sv;
        mbar_arrive_expect_tx(&bar[NBUF], bytes);
        seg_issue(vst(0), vin + in.offs, sv, &bar[NBUF], pol);
    };
    if (tid == 0) {
        for (int b = 0; b < NBUF + (VS ? 1 : 0); ++b) mbar_init(&bar[b], 1);
        mbar_fence_init();
        for (int b = 0; b < NBUF; ++b) issue(b, atomicAdd(&prm.ctl->claim[prm.p], 1u));
        if constexpr (VS) vissue(info[0]);
    }
    __syncthreads();

    const int lo = prm.lo;
    const uint32_t mask = prm.mask;
    const uint32_t ltm = lanemask_lt();
    // per-digit destination base of a tile relative to its bucket: sub-bucket start + counts
    // of the earlier tiles of the bucket (tile order = memory order: stable), loaded a tile
    // ahead (two buffers) or before the wait for the tile's data (one buffer)
    uint32_t m0 = 0, m1 = 0, m2 = 0;
    uint64_t boffs = 0, mdst = 0;
    auto meta_load = [&](const StageInfo &in) {
        if (in.valid) {
            if (tid < RADIX) {
                if constexpr (DST) mdst = tid <= static_cast<int>(prm.mask) ? prm.dst_off[tid] : 0ull;
                else m0 = prm.sub_rel[static_cast<uint64_t>(in.bucket) * RADIX + tid];
                m1 = prm.tile_pref[static_cast<uint64_t>(in.tile) * RADIX + tid];
                m2 = in.carry_row != EMPTY_RANGE ? prm.carry[static_cast<uint64_t>(in.carry_row) * RADIX + tid] : 0u;
            }
            boffs = prm.buckets[in.bucket].offs;
        }
    };
    meta_load(info[0]);
    for (uint32_t it = 0;; ++it) {
        const int s = static_cast<int>(it % NBUF);
        const uint32_t par = (it / NBUF) & 1u;
        const StageInfo in = info[s];
        if (!in.valid) break;
        const uint32_t count = in.count;
        const uint32_t gbase = m0 + m1 + m2;  // thread tid = digit tid
        const uint64_t gdst = mdst;
        const uint64_t tboffs = boffs;
        Seg sk, sv;
        sk.pad = in.kpad;
        sk.i0 = static_cast<int32_t>(in.k0);
        sk.i1 = static_cast<int32_t>(in.k1);
        sv.pad = in.vpad;
        sv.i0 = static_cast<int32_t>(in.v0);
        sv.i1 = static_cast<int32_t>(in.v1);
        const K *ksrc = kin_of(in.src) + in.offs;
        const VT *vsrc = HV ? vin_of(in.src) + in.offs : nullptr;
        K *const ks = kst(s);
        VT *const vs = HV ? vst(VS ? 0 : s) : nullptr;
        mbar_wait(&bar[s], par);
        const bool full = count == static_cast<uint32_t>(L::KPB) && seg_full(sk, count) && (!HV || VS || seg_full(sv, count));
        const bool mapin = TY && prm.kind != 0 && in.src == SRC_IN;     // records still in the input
        const bool unmap = TY && prm.kind != 0 && prm.final_pass != 0;  // their final place
        const VT *vb = HV ? vs + sv.pad : nullptr;
        // VS: wait for this tile's values (issued after the previous tile's write-out)
        auto vwait = [&]() {
            if constexpr (VS) {
                mbar_wait(&bar[NBUF], it & 1u);
                const Seg s2 = *vinfo;
                vb = vs + s2.pad;
                if (!seg_full(s2, count)) {  // (only at the ends of the buffer)
                    seg_fill_edges<VT, THREADS>(vs, vsrc, s2, count);
                    __syncthreads();
                }
            }
        };

        auto body = [&](auto full_tag) {
            constexpr bool FULL = decltype(full_tag)::value;
            // the values of the elements the bulk copy did not cover (segments at the ends
            // of the buffer) into shared memory, read by the write-out after the barriers
            constexpr bool DIRECT = HRS_SC_DIRECT && HV;
            if (!DIRECT && !VS && !FULL && HV) seg_fill_edges<VT, THREADS>(vs, vsrc, sv, count);
            const K *const kb = ks + sk.pad;
            [[maybe_unused]] VT val[DIRECT ? KPT : 1];
            // the keys stay in registers from here to the placement; the in-warp ranks are
            // packed two to a register (rank < 32 * KPT < 2^16), the digits recomputed
            constexpr int NR = (KPT + 1) / 2;
            K key[KPT];
            uint32_t rk[NR];
            uint32_t valid = 0;  // bit c: element wbase + c*32 + lane exists
#pragma unroll
            for (int c = 0; c < KPT; ++c) {
                const uint32_t e = wbase + c * 32 + lane;
                const bool v = FULL || e < count;
                key[c] = v ? (FULL ? kb[e] : seg_get(ks, ksrc, sk, e)) : K(0);
                if (mapin) key[c] = key_map(key[c], prm.kind, false);
                if constexpr (DIRECT) val[c] = v ? (FULL ? vb[e] : seg_get(vs, vsrc, sv, e)) : VT(0);
                valid |= v ? (1u << c) : 0u;
            }
#pragma unroll
            for (int i = 0; i < NR; ++i) rk[i] = 0;
            auto dig = [&](int c) -> uint32_t { return digit_of(key[c], lo, mask); };
            // ---- A: in-warp ranks
            auto count_fast = [&]() {
#pragma unroll
                for (int c = 0; c < KPT; ++c)
                    if (valid & (1u << c)) rk[c >> 1] |= atomicAdd(&ca[dig(c)], 1u) << (16 * (c & 1));
            };
            auto count_exact = [&]() {
#pragma unroll
                for (int c = 0; c < KPT; ++c) {
                    const bool v0 = (valid >> c) & 1u;
                    const uint32_t d0 = v0 ? dig(c) : 0u;
                    const uint32_t p0 = v0 ? ca[d0] : 0u;
                    __syncwarp();
                    if (v0) atomicAdd(&ca[d0], 1u);
                    __syncwarp();
                    const uint32_t k0 = v0 ? ca[d0] - p0 : 0u;
                    const uint32_t m = __match_any_sync(0xffffffffu, k0 > 1 ? d0 : 0xFFFFFFFFu);
                    if (v0) rk[c >> 1] |= (p0 + (k0 > 1 ? __popc(m & ltm) : 0u)) << (16 * (c & 1));
                }
            };
            // ---- B: fold the warp counters into first slots; digit starts and bases
            auto fold = [&]() {
                __syncthreads();  // counts complete
                // (the W counters of digit tid are read twice rather than kept: registers)
                uint32_t t = 0, incl = 0;
                if (tid < RADIX) {
#pragma unroll
                    for (int w = 0; w < W; ++w) t += cnt[w * RADIX + tid];
                    incl = t;
#pragma unroll
                    for (int o = 1; o < 32; o <<= 1) {
                        const uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
                        if (lane >= o) incl += y;
                    }
                    if (lane == 31) wsum[warp] = incl;
                }
                __syncthreads();
                if (tid < RADIX) {
                    uint32_t run = incl - t;
#pragma unroll
                    for (int w = 0; w < RADIX / 32; ++w) run += w < warp ? wsum[w] : 0u;
                    if constexpr (DST) {
                        // element offset of slot 0 of digit d (mod 2^64: slot `run` onward is in range)
                        const uint64_t v = (gdst & DST_OFF_MASK) + gbase - static_cast<uint64_t>(run);
                        gs[tid] = make_uint2(static_cast<uint32_t>(v), static_cast<uint32_t>(v >> 32));
                        sstart[tid] = run | (static_cast<uint32_t>(gdst >> 48) << 16);  // start | window << 16
                    } else if constexpr (L::PTR) {
                        // byte address of the destination of slot 0 of digit d (slot `run`
                        // onward is in range)
                        const unsigned long long a = reinterpret_cast<unsigned long long>(kout) +
                            static_cast<unsigned long long>(static_cast<long long>(tboffs) + static_cast<long long>(gbase) -
                                                            static_cast<long long>(run)) * sizeof(K);
                        reinterpret_cast<uint4 *>(gs)[tid] = make_uint4(static_cast<uint32_t>(a), static_cast<uint32_t>(a >> 32), run, 0u);
                    } else {
                        gs[tid] = make_uint2(gbase - run, run);
                    }
#pragma unroll
                    for (int w = 0; w < W; ++w) {
                        const uint32_t x = cnt[w * RADIX + tid];
                        cnt[w * RADIX + tid] = run;
                        run += x;
                    }
                }
                __syncthreads();  // first slots published
            };
            // ---- C: place keys and element indices at their slots (in place: every key
            // of the tile was read into registers before the fold's barriers); clear the
            // warp's counters for the next rank
            auto place = [&]() {
#pragma unroll
                for (int c = 0; c < KPT; ++c) {
                    if (valid & (1u << c)) {
                        const uint32_t slot = ca[dig(c)] + ((rk[c >> 1] >> (16 * (c & 1))) & 0xFFFFu);
                        ks[slot] = key[c];
                        if constexpr (DIRECT) vs[slot] = val[c];
                        else sidx[slot] = static_cast<uint16_t>(wbase + c * 32 + lane);
                    }
                }
                __syncwarp();
#pragma unroll
                for (int d = lane; d < RADIX; d += 32) ca[d] = 0;
                __syncthreads();  // sorted tile complete
            };
            // ---- D: write-out (check: the complete stability condition)
            K *const kdst = kout + tboffs;
            VT *const vdst = HV ? vout + tboffs : nullptr;
            auto write_out = [&](bool check) -> bool {
                bool bad = false;
                if constexpr (L::PTR) {
                    // the value's address is the key's plus the (uniform) distance between the
                    // output arrays; a slot whose element index is below its predecessor's in
                    // the same digit run sets the top bit of badw
                    const long long vdelta = HV ? reinterpret_cast<const char *>(vout) - reinterpret_cast<const char *>(kout) : 0;
                    uint32_t badw = 0;
                    const uint4 *gp = reinterpret_cast<const uint4 *>(gs);
#pragma unroll (WO_UNROLL)
                    for (int c = 0; c < KPT; ++c) {
                        const uint32_t j = c * THREADS + tid;
                        if (FULL || j < count) {
                            const K k = ks[j];
                            const uint4 g = gp[digit_of(k, lo, mask)];
                            K *const kp = reinterpret_cast<K *>((static_cast<unsigned long long>(g.y) << 32) | g.x) + j;
                            *kp = unmap ? key_map(k, prm.kind, true) : k;
                            const uint32_t i = sidx[j];
                            if constexpr (HV) *reinterpret_cast<VT *>(reinterpret_cast<char *>(kp) + vdelta) = vb[i];
                            if (check) badw |= i - (j > g.z ? static_cast<uint32_t>(sidx[j - 1]) : 0u);
                        }
                    }
                    return (badw >> 31) != 0u;
                }
#pragma unroll (WO_UNROLL)
                for (int c = 0; c < KPT; ++c) {
                    const uint32_t j = c * THREADS + tid;
                    if (FULL || j < count) {
                        const K k = ks[j];
                        if constexpr (DST) {
                            const uint32_t i = sidx[j];
                            const uint32_t d = digit_of(k, lo, mask);
                            const uint2 g = gs[d];
                            const uint32_t sw = sstart[d];
                            const uint64_t pos = ((static_cast<uint64_t>(g.y) << 32) | g.x) + j;
                            const uint32_t w = sw >> 16;
                            reinterpret_cast<K *>(prm.dst_kwin[w])[pos] = k;
                            if (HV) reinterpret_cast<VT *>(prm.dst_vwin[w])[pos] = vb[i];
                            if (check && j > (sw & 0xFFFFu)) bad |= sidx[j - 1] > i;
                        } else if constexpr (DIRECT) {
                            const uint32_t pos = gs[digit_of(k, lo, mask)].x + j;
                            kdst[pos] = unmap ? key_map(k, prm.kind, true) : k;
                            vdst[pos] = vs[j];
                        } else {
                            const uint32_t i = sidx[j];
                            const uint2 g = gs[digit_of(k, lo, mask)];
                            const uint32_t pos = g.x + j;
                            if constexpr (HRS_SC_STHINT && sizeof(K) == 4 && (!HV || sizeof(VT) == 4)) {
                                if (sthint) {
                                    st_hint(reinterpret_cast<uint32_t *>(kdst + pos), static_cast<uint32_t>(unmap ? key_map(k, prm.kind, true) : k), spol);
                                    if (HV) st_hint(reinterpret_cast<uint32_t *>(vdst + pos), static_cast<uint32_t>(vb[i]), spol);
                                    if (check && j > g.y) bad |= sidx[j - 1] > i;
                                    continue;
                                }
                            }
                            kdst[pos] = unmap ? key_map(k, prm.kind, true) : k;
                            if (HV) vdst[pos] = vb[i];
                            if (check && j > g.y) bad |= sidx[j - 1] > i;
                        }
                    }
                }
                return bad;
            };
            // contention probe: equal digits among the 5 butterfly partners of column 0
            // (a uniform digit gives 0.6 on average over the warp): heavy contention makes
            // returning atomics slow, and the exact rank cheap
            bool fast;
            {
                const uint32_t d0 = (valid & 1u) ? dig(0) : INVALID_DIGIT;
                uint32_t eq = 0;
#pragma unroll
                for (int k2 = 1; k2 < 32; k2 <<= 1) eq += __shfl_xor_sync(0xffffffffu, d0, k2) == d0;
                fast = __reduce_add_sync(0xffffffffu, eq) < 8;
            }
            if (fast) count_fast();
            else count_exact();
            fold();
            place();
            // the next tile's metadata (info[s ^ 1] was published by the issue after the
            // previous tile, before this tile's barriers); the loads overlap the write-out
            if (NBUF == 2) meta_load(info[s ^ 1]);
            vwait();
            const bool bad = write_out(fast && !DIRECT);
            if (__syncthreads_or(bad || (fast && prm.force_redo))) {
                // the atomics did not serve the lanes of a warp in order: rank the tile
                // again with the rank that is stable by construction (same digit totals, so
                // the starts and bases are unchanged) and write it out again
                if (tid == 0) atomicAdd(&prm.ctl->redo, 1ull);
#pragma unroll
                for (int i = 0; i < NR; ++i) rk[i] = 0;
                count_exact();
                fold();
                place();
                write_out(false);
                __syncthreads();
            }
        };
        if (full) body(std::true_type{});
        else body(std::false_type{});
        // ---- the staging buffer is free again (barrier above): claim the next tile into it
        if (tid == 0) {
            fence_proxy_async();
            if constexpr (VS) vissue(info[s ^ 1]);
            issue(s, atomicAdd(&prm.ctl->claim[prm.p], 1u));
        }
        if (NBUF == 1) {
            __syncthreads();  // info[0] of the next tile
            meta_load(info[0]);
        }
    }
}

// ------------------------------------------------------------------ local sort

struct LocalParams {
    uint64_t n;  // elements of the buffers
    const void *src_keys[3];  // indexed by SrcCode
    const void *src_vals[3];
    void *keys_out;
    void *vals_out;
    const LocalEntry *list;
    const uint32_t *count;  // entries in the list
    LocalEntry *fb_list;    // k_local_cnt: entries handed to the narrow k_local
    uint32_t *fb_count;
    uint32_t fb_cap;
    // narrow k_local: entries handed to the wide variant, one list per wide configuration
    // (class wide_cfg(size class)); wide_single >= 0: the single-configuration ablation
    LocalEntry *wide_list[HRS_NUM_CLASSES];
    uint32_t *wide_count;
    uint32_t wide_cap[HRS_NUM_CLASSES];
    int wide_single;
    int wide_top;  // largest wide configuration
    int begin_bit;
    int force_redo;  // HRS_FLAG_FORCE_REDO: every stability check of the fast rank fails
    unsigned long long *redo;  // Ctl::redo
    int kind;        // hrs_key_kind: keys read from the input are mapped, every write is final (unmapped)
};

// Shared memory of one local-sort CTA: NSTAGE staging buffers {keys, values}; after
// the keys have been read into registers the key buffer doubles as the buffer of
// the LSD passes, which move (key, 16-bit index) pairs; the values are gathered from
// their staging buffer once, at the end.
// Composite word of the local sort.  The narrow variant ranks 32-bit composites
// (top <= 19 sort bits << 13 | index) and resolves ties of the top bits afterwards;
// the wide variant (entries the narrow one hands over) ranks 64-bit composites for
// 32-bit keys and (key, 16-bit index) pairs for 64-bit keys.
// WIDE = 2 is the narrow variant for begin_bit == 0: entries of at most 19 sort bits
// rank their composites inside the key staging buffer and rebuild the keys from the
// composite and the bucket's common high bits (no key gather, no composite buffer);
// entries with more sort bits go straight to the wide variant.
template <typename K, int WIDE>
struct LocalWord {
    using CT = typename std::conditional<WIDE == 1, unsigned long long, uint32_t>::type;
    static constexpr bool PAIRS = WIDE == 1 && sizeof(K) == 8;
    static constexpr bool RECON = WIDE == 2;
    static constexpr size_t buf_bytes = RECON ? 0 : (PAIRS ? sizeof(uint16_t) : sizeof(CT));
};

template <typename K, typename V, int THREADS, int KPT, int NSTAGE, int WIDE = 0>
struct LocalSmem {
    static constexpr int W = THREADS / 32;
    static constexpr int CAP = THREADS * KPT;
    using VT = ValT<V>;
    static constexpr bool HV = HasVal<V>::value;
    static constexpr size_t off_bar = 0;
    static constexpr size_t off_info = align16(sizeof(uint64_t) * NSTAGE);
    using RK = Ranker<THREADS, KPT>;
    static constexpr size_t off_rank = align16(off_info + sizeof(uint32_t) * 16 * (NSTAGE + 1));
    static constexpr size_t off_red = align16(off_rank + RK::smem_bytes);
    // composite buffer (or the 16-bit index buffer of the pair path)
    static constexpr size_t off_sidx = align16(off_red + sizeof(K) * 2 * W);
    static constexpr size_t off_kst = align16(off_sidx + LocalWord<K, WIDE>::buf_bytes * CAP);
    static constexpr size_t kst_bytes = align16(sizeof(K) * (CAP + 32 / sizeof(K)));
    static constexpr size_t off_vst = off_kst + NSTAGE * kst_bytes;
    static constexpr size_t vst_bytes = HV ? align16(sizeof(VT) * (CAP + 32 / sizeof(VT))) : 0;
    static constexpr size_t bytes = off_vst + NSTAGE * vst_bytes;
};

__device__ __forceinline__ uint32_t warp_and(uint32_t x) { return __reduce_and_sync(0xffffffffu, x); }
__device__ __forceinline__ uint32_t warp_or(uint32_t x) { return __reduce_or_sync(0xffffffffu, x); }
__device__ __forceinline__ unsigned long long warp_and(unsigned long long x) {
    const uint32_t lo = __reduce_and_sync(0xffffffffu, static_cast<uint32_t>(x));
    const uint32_t hi = __reduce_and_sync(0xffffffffu, static_cast<uint32_t>(x >> 32));
    return (static_cast<unsigned long long>(hi) << 32) | lo;
}
__device__ __forceinline__ unsigned long long warp_or(unsigned long long x) {
    const uint32_t lo = __reduce_or_sync(0xffffffffu, static_cast<uint32_t>(x));
    const uint32_t hi = __reduce_or_sync(0xffffffffu, static_cast<uint32_t>(x >> 32));
    return (static_cast<unsigned long long>(hi) << 32) | lo;
}

template <typename K, typename V, int THREADS, int KPT, int NSTAGE, int MINB, int WIDE, bool TY>
__global__ void __launch_bounds__(THREADS, MINB) k_local(LocalParams prm) {
    pdl_wait();
    using L = LocalSmem<K, V, THREADS, KPT, NSTAGE, WIDE>;
    using LW = LocalWord<K, WIDE>;
    using CT = typename LW::CT;
    constexpr int IB = 13;  // index bits: CAP <= 8192
    static_assert(L::CAP <= (1 << IB), "local-sort capacity exceeds the composite index");
    constexpr int W = THREADS / 32;
    constexpr bool HV = HasVal<V>::value;
    using VT = ValT<V>;
    extern __shared__ __align__(16) unsigned char smem[];
    uint64_t *bar = reinterpret_cast<uint64_t *>(smem + L::off_bar);
    uint32_t *info = reinterpret_cast<uint32_t *>(smem + L::off_info);  // [s][16]
    typename L::RK ranker;
    ranker.init(reinterpret_cast<uint32_t *>(smem + L::off_rank));
    K *red = reinterpret_cast<K *>(smem + L::off_red);
    uint16_t *sidx = reinterpret_cast<uint16_t *>(smem + L::off_sidx);
    auto kst = [&](int s) { return reinterpret_cast<K *>(smem + L::off_kst + s * L::kst_bytes); };
    auto vst = [&](int s) { return reinterpret_cast<VT *>(smem + L::off_vst + s * L::vst_bytes); };
    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    const uint32_t nent = *prm.count;
    if (blockIdx.x >= nent) return;
    K *__restrict__ kout = static_cast<K *>(prm.keys_out);
    VT *__restrict__ vout = static_cast<VT *>(prm.vals_out);
    const uint64_t pol = policy_evict_first();
    const int begin_bit = prm.begin_bit;
    const uint32_t ltm = lanemask_lt();

    auto srck = [&](uint32_t code) -> const K * {
        return static_cast<const K *>(code == SRC_IN    ? prm.src_keys[SRC_IN]
                                      : code == SRC_AUX ? prm.src_keys[SRC_AUX]
                                                        : prm.src_keys[SRC_OUT]);
    };
    auto srcv = [&](uint32_t code) -> const VT * {
        return static_cast<const VT *>(code == SRC_IN    ? prm.src_vals[SRC_IN]
                                       : code == SRC_AUX ? prm.src_vals[SRC_AUX]
                                                         : prm.src_vals[SRC_OUT]);
    };
    // the recon variant hands entries of more than 19 sort bits to the wide variant
    // hand an entry to the wide variant's list of its size
    auto to_wide = [&](const LocalEntry &en) {
        const int w = prm.wide_single >= 0 ? prm.wide_single : wide_cfg(size_class_of(en.count), prm.wide_top, sizeof(K) == 8);
        const uint32_t slot = atomicAdd(&prm.wide_count[w], 1u);
        if (slot < prm.wide_cap[w]) prm.wide_list[w][slot] = en;
    };
    // RECON takes at most 19 sort bits (the composite); with HRS_WIDE64 the narrow
    // variant for 64-bit keys passes entries of more sort bits straight to the wide one
    constexpr bool DIRECT = LW::RECON || (HRS_WIDE64 && WIDE == 0 && sizeof(K) == 8);
    auto mine = [&](const LocalEntry &en) {
        if (!DIRECT || static_cast<int>(en.hi_bit) - prm.begin_bit <= 32 - IB) return true;
        to_wide(en);
        return false;
    };
    __shared__ uint32_t s_fallback;
    // info[s]: 0 entry, 1 count, 2 hi_bit, 3 src, 4..5 offs, 6..8 key seg, 9..11 value seg, 12 next stride
    auto issue = [&](int s, uint32_t e) {
        uint32_t *in = info + 16 * s;
        LocalEntry en;
        while (e < nent) {  // grid-stride over the entries of this variant
            en = prm.list[e];
            if (mine(en)) break;
            e += gridDim.x;
        }
        in[0] = e;
        if (e >= nent) {
            mbar_arrive_expect_tx(&bar[s], 0);  // completes the phase: the waiters see the end
            return;
        }
        in[1] = en.count;
        in[2] = en.hi_bit;
        in[3] = en.src;
        in[4] = static_cast<uint32_t>(en.offs);
        in[5] = static_cast<uint32_t>(en.offs >> 32);
        Seg sk, sv;
        const K *kbuf = srck(en.src);
        const K *ks = kbuf + en.offs;
        uint32_t bytes = seg_plan(ks, en.count, kbuf, kbuf + prm.n, sk);
        in[6] = sk.pad;
        in[7] = static_cast<uint32_t>(sk.i0);
        in[8] = static_cast<uint32_t>(sk.i1);
        const VT *vs = nullptr;
        if (HV) {
            const VT *vbuf = srcv(en.src);
            vs = vbuf + en.offs;
            bytes += seg_plan(vs, en.count, vbuf, vbuf + prm.n, sv);
            in[9] = sv.pad;
            in[10] = static_cast<uint32_t>(sv.i0);
            in[11] = static_cast<uint32_t>(sv.i1);
        }
        mbar_arrive_expect_tx(&bar[s], bytes);
        seg_issue(kst(s), ks, sk, &bar[s], pol);
        if (HV) seg_issue(vst(s), vs, sv, &bar[s], pol);
    };
    if (tid == 0) {
        for (int s = 0; s < NSTAGE; ++s) mbar_init(&bar[s], 1);
        mbar_fence_init();
        uint32_t e = blockIdx.x;
        for (int s = 0; s < NSTAGE; ++s) {
            issue(s, e);
            e = info[16 * s] + gridDim.x;
        }
        info[16 * NSTAGE] = e;  // next entry to look at
    }
    __syncthreads();

    for (uint32_t it = 0;; ++it) {
        const int s = static_cast<int>(it % NSTAGE);
        const uint32_t par = (it / NSTAGE) & 1u;
        const uint32_t *in = info + 16 * s;
        // the producer wrote info[s] before its arrive on bar[s]: the wait acquires it
        mbar_wait(&bar[s], par);
        const uint32_t e_id = in[0];
        if (e_id >= nent) break;
        const uint32_t count = in[1];
        const int hi_bit = static_cast<int>(in[2]);
        const uint32_t src = in[3];
        // signed / float keys (hrs_sort_typed): keys read from the input are mapped to their
        // order-preserving image, every key this kernel writes is final and mapped back
        const bool typed = TY && prm.kind != 0;
        const bool mapin = typed && src == SRC_IN;
        auto kin_map = [&](K x) -> K { return mapin ? key_map(x, prm.kind, false) : x; };
        auto kout_map = [&](K x) -> K { return typed ? key_map(x, prm.kind, true) : x; };
        // a staged key copied to the output: the original if it came from the input
        auto kout_raw = [&](K x) -> K { return (typed && !mapin) ? key_map(x, prm.kind, true) : x; };
        const uint64_t offs = static_cast<uint64_t>(in[4]) | (static_cast<uint64_t>(in[5]) << 32);
        Seg sk, sv;
        sk.pad = in[6];
        sk.i0 = static_cast<int32_t>(in[7]);
        sk.i1 = static_cast<int32_t>(in[8]);
        sv.pad = in[9];
        sv.i0 = static_cast<int32_t>(in[10]);
        sv.i1 = static_cast<int32_t>(in[11]);
        const K *ksrc = srck(src) + offs;
        const VT *vsrc = HV ? srcv(src) + offs : nullptr;
        K *ks = kst(s);
        VT *vs = HV ? vst(s) : nullptr;
        // the entry may be sorted in place: elements the bulk copy did not cover (entries
        // at the ends of the buffer) go into shared memory now, before any thread writes
        // the output; they are read through seg_get until the next barrier
        seg_fill_edges<K, THREADS>(ks, ksrc, sk, count);
        if (HV) seg_fill_edges<VT, THREADS>(vs, vsrc, sv, count);
        // BAL: every warp takes kpt = ceil(count / THREADS) columns, so the work is spread
        // over all warps whatever the bucket size (element e = warp*32*kpt + c*32 + lane);
        // otherwise kpt = KPT and warps past the end of the bucket idle
        constexpr bool BAL = HRS_EXP == 10 || HRS_EXP == 12;
        const int kpt = BAL ? static_cast<int>(min((count + THREADS - 1) / THREADS, static_cast<uint32_t>(KPT))) : KPT;
        const uint32_t wbase = static_cast<uint32_t>(warp) * 32u * kpt;
        K key[KPT];
        uint32_t idx[KPT];
        K a = ~K(0), o = K(0);
#pragma unroll
        for (int c = 0; c < KPT; ++c) {
            const uint32_t e = wbase + c * 32 + lane;
            idx[c] = e;
            key[c] = kin_map((!BAL || c < kpt) ? (e < count ? seg_get(ks, ksrc, sk, e) : ks[sk.pad + e]) : K(0));  // past count: stale, never written out
            const bool v = (!BAL || c < kpt) && e < count;
            a &= v ? key[c] : ~K(0);
            o |= v ? key[c] : K(0);
        }
        // bits that vary across the bucket: digits where they are all equal are skipped
        a = warp_and(a);
        o = warp_or(o);
        if (lane == 0) {
            red[warp] = a;
            red[W + warp] = o;
        }
        __syncthreads();
        K diff = 0, kconst = 0;
        {
            K aa = ~K(0), oo = K(0);
#pragma unroll
            for (int w = 0; w < W; ++w) {
                aa &= red[w];
                oo |= red[W + w];
            }
            diff = aa ^ oo;
            kconst = aa;  // the bits of positions where diff == 0 are common to all keys
        }
        const bool active = wbase < count;
        bool moved = false;
        const int sb = hi_bit - begin_bit;
        if constexpr (!LW::PAIRS) {
            // ---- composite path: one word per record, composite = (top sort bits << IB) | index.
            // The LSD passes move composites only; keys and values are gathered from the
            // staging buffers through the index at the end (the key bits outside the
            // sorted range are carried that way too).  The narrow variant keeps the top
            // TB <= 19 sort bits and then orders the runs of records that tie on them by
            // the remaining bits (insertion sort; a bucket with a run longer than RUN_MAX
            // is handed to the wide variant).
            constexpr int CB = static_cast<int>(8 * sizeof(CT)) - IB;  // sort bits a composite holds
            constexpr uint32_t RUN_MAX = 16;
            const int tb = sb < CB ? sb : CB;
            const int tlo = hi_bit - tb;  // composite field = key bits [tlo, hi_bit)
            // recon: the keys are in registers, their staging buffer holds the composites
            CT *comp = LW::RECON ? reinterpret_cast<CT *>(ks) : reinterpret_cast<CT *>(sidx);
            const CT tmask = tb >= static_cast<int>(8 * sizeof(CT)) ? ~CT(0) : ((CT(1) << tb) - 1);
            CT cv[KPT];
#pragma unroll
            for (int c = 0; c < KPT; ++c)
                cv[c] = ((static_cast<CT>(key[c] >> tlo) & tmask) << IB) | static_cast<CT>(idx[c]);
            const CT cdiff = (static_cast<CT>(diff >> tlo) & tmask) << IB;
            // LSD passes over the composites, with the fast rank first (fast = true)
            auto passes = [&](bool fast) {
                for (int lo = IB; lo < IB + tb; lo += 8) {
                    const int width = min(8, IB + tb - lo);
                    const uint32_t mask = (1u << width) - 1u;
                    if ((static_cast<uint32_t>(cdiff >> lo) & mask) == 0) continue;  // constant digit: identity pass
                    moved = true;
                    // padding slots (e >= count) carry digit 256: they rank after every record
                    // and end up in slots >= count again, so no per-element guards are needed
                    uint32_t dg[KPT];
#pragma unroll
                    for (int c = 0; c < KPT; ++c)
                        dg[c] = (wbase + c * 32 + lane) < count ? digit_of(cv[c], lo, mask) : INVALID_DIGIT;
                    ranker.rank(dg, kpt, active, ltm, fast);
                    if (active) {
#pragma unroll
                        for (int c = 0; c < KPT; ++c)
                            if (!BAL || c < kpt) comp[dg[c]] = cv[c];
                    }
                    __syncthreads();
                    if (active) {
#pragma unroll
                        for (int c = 0; c < KPT; ++c)
                            if (!BAL || c < kpt) cv[c] = comp[wbase + c * 32 + lane];
                    }
                }
            };
            // more sort bits than the composite holds: the tie runs on the top bits are
            // sorted by insertion afterwards, and a run longer than RUN_MAX sends the
            // bucket to the wide variant.  AND-skewed keys make the all-zero top field
            // such a run: count it first and hand the bucket over before any pass.
            bool early = false;
            if (!LW::RECON && sb > tb) {
                uint32_t z = 0;
#pragma unroll
                for (int c = 0; c < KPT; ++c)
                    z += ((!BAL || c < kpt) && wbase + c * 32 + lane < count && (cv[c] >> IB) == 0) ? 1u : 0u;
                z = __reduce_add_sync(0xffffffffu, z);
                if (tid == 0) s_fallback = 0;
                __syncthreads();
                if (lane == 0 && z) atomicAdd(&s_fallback, z);
                __syncthreads();
                early = s_fallback > RUN_MAX;
            }
            if (!early) passes(true);
            if (!early && moved) {
                // the composites are distinct (index field), so the passes were all stable
                // iff they end strictly increasing; otherwise put every composite back at
                // its index and redo the passes with the rank that is stable by construction
                bool bad = false;
                if (active) {
#pragma unroll
                    for (int c = 0; c < KPT; ++c) {
                        const uint32_t e = wbase + c * 32 + lane;
                        if ((!BAL || c < kpt) && e > 0 && e < count) bad |= comp[e - 1] >= cv[c];
                    }
                }
                if (__syncthreads_or(bad || prm.force_redo)) {
                    if (tid == 0) atomicAdd(prm.redo, 1ull);
                    if (active) {
#pragma unroll
                        for (int c = 0; c < KPT; ++c)
                            if (!BAL || c < kpt) comp[static_cast<uint32_t>(cv[c]) & ((1u << IB) - 1u)] = cv[c];
                    }
                    __syncthreads();
                    if (active) {
#pragma unroll
                        for (int c = 0; c < KPT; ++c)
                            if (!BAL || c < kpt) cv[c] = comp[wbase + c * 32 + lane];
                    }
                    passes(false);
                }
            }
            const K *const ksp = ks + sk.pad;
            bool fallback = early;
            if (!early && !LW::RECON && sb > tb) {
                // ---- runs that tie on the top bits: insertion sort by (low bits, index);
                // inside a run the records are in index order (the passes are stable), so
                // shifting only past strictly greater low bits keeps the sort stable
                if (!moved) {
                    // comp was not written: store the (unsorted) composites
#pragma unroll
                    for (int c = 0; c < KPT; ++c)
                        if ((!BAL || c < kpt) && active) comp[wbase + c * 32 + lane] = cv[c];
                }
                // a run longer than RUN_MAX exists iff some slot e has the same top bits as
                // slot e + RUN_MAX (the slots are sorted by them): then the bucket goes to
                // the wide variant without any insertion sort
                bool longrun = false;
                for (uint32_t e = tid; e + RUN_MAX < count; e += THREADS)
                    longrun |= (comp[e] >> IB) == (comp[e + RUN_MAX] >> IB);
                if (tid == 0) s_fallback = 0;
                if (__syncthreads_or(longrun)) {
                    if (tid == 0) s_fallback = 1;
                    __syncthreads();
                }
                const int lb = sb - tb;
                const K lmask = lb >= static_cast<int>(8 * sizeof(K)) ? ~K(0) : ((K(1) << lb) - 1);
                auto low = [&](CT x) -> K {
                    return (kin_map(ksp[static_cast<uint32_t>(x) & ((1u << IB) - 1u)]) >> begin_bit) & lmask;
                };
                for (uint32_t e = tid; e + 1 < count && !s_fallback; e += THREADS) {
                    const CT t = comp[e] >> IB;
                    if ((comp[e + 1] >> IB) != t) continue;
                    if (e > 0 && (comp[e - 1] >> IB) == t) continue;  // not the start of the run
                    uint32_t r = 2;
                    while (e + r < count && (comp[e + r] >> IB) == t) ++r;
                    if (r > RUN_MAX) {
                        s_fallback = 1;
                        continue;
                    }
                    for (uint32_t i = 1; i < r; ++i) {
                        const CT x = comp[e + i];
                        const K lx = low(x);
                        int j = static_cast<int>(i) - 1;
                        while (j >= 0) {
                            const CT y = comp[e + j];
                            if (low(y) <= lx) break;
                            comp[e + j + 1] = y;
                            --j;
                        }
                        comp[e + j + 1] = x;
                    }
                }
                __syncthreads();
                fallback = s_fallback != 0;
                moved = true;
                if (!fallback && active) {
#pragma unroll
                    for (int c = 0; c < KPT; ++c)
                        if (!BAL || c < kpt) cv[c] = comp[wbase + c * 32 + lane];
                }
            }
            if (fallback) {
                if (tid == 0) {
                    LocalEntry en;
                    en.offs = offs;
                    en.count = count;
                    en.hi_bit = static_cast<uint16_t>(hi_bit);
                    en.src = static_cast<uint16_t>(src);
                    to_wide(en);
                }
            } else if (moved || src != SRC_OUT || typed) {
                K *const kd = kout + offs;
                VT *const vd = HV ? vout + offs : nullptr;
                const VT *const vsp = HV ? vs + sv.pad : nullptr;
                // recon (begin_bit == 0, all sort bits in the composite): key = common bits
                // above hi_bit | the composite's sort field
                const K khigh = hi_bit >= static_cast<int>(8 * sizeof(K)) ? K(0) : (kconst & ~((K(1) << hi_bit) - 1));
#pragma unroll
                for (int c = 0; c < KPT; ++c) {
                    const uint32_t e = wbase + c * 32 + lane;
                    if ((!BAL || c < kpt) && e < count) {
                        const uint32_t ix = static_cast<uint32_t>(cv[c]) & ((1u << IB) - 1u);
                        kd[e] = LW::RECON ? kout_map(khigh | static_cast<K>(static_cast<uint32_t>(cv[c]) >> IB))
                                          : kout_raw(ksp[ix]);
                        if (HV) vd[e] = vsp[ix];
                    }
                }
            }
        } else {
            // ---- pair path (64-bit keys, wide variant): (key, index) pairs, the key
            // staging buffer doubles as the sort buffer.  The passes use the fast rank;
            // the result is the stable sort iff (sort bits, index) strictly increase along
            // the slots, else the passes are redone from the source with the exact rank.
            K *skeys = ks;
            auto pair_passes = [&](bool fast) {
            for (int lo = begin_bit; lo < hi_bit; lo += 8) {
                const int width = min(8, hi_bit - lo);
                const uint32_t mask = (1u << width) - 1u;
                if ((static_cast<uint32_t>(diff >> lo) & mask) == 0) continue;  // constant digit: identity pass
                moved = true;
                uint32_t dg[KPT];
#pragma unroll
                for (int c = 0; c < KPT; ++c)
                    dg[c] = (wbase + c * 32 + lane) < count ? digit_of(key[c], lo, mask) : INVALID_DIGIT;
                ranker.rank(dg, kpt, active, ltm, fast);
                if (active) {
#pragma unroll
                    for (int c = 0; c < KPT; ++c) {
                        if (!BAL || c < kpt) {
                            skeys[dg[c]] = key[c];
                            sidx[dg[c]] = static_cast<uint16_t>(idx[c]);
                        }
                    }
                }
                __syncthreads();
                if (active) {
#pragma unroll
                    for (int c = 0; c < KPT; ++c) {
                        if (!BAL || c < kpt) {
                            const uint32_t e = wbase + c * 32 + lane;
                            key[c] = skeys[e];
                            idx[c] = sidx[e];
                        }
                    }
                }
            }
            };
            pair_passes(true);
            if (moved) {
                const K smask = sb >= static_cast<int>(8 * sizeof(K)) ? ~K(0) : ((K(1) << sb) - 1);
                bool bad = false;
                if (active) {
#pragma unroll
                    for (int c = 0; c < KPT; ++c) {
                        const uint32_t e = wbase + c * 32 + lane;
                        if ((!BAL || c < kpt) && e > 0 && e < count) {
                            const K pa = (skeys[e - 1] >> begin_bit) & smask, pb = (key[c] >> begin_bit) & smask;
                            bad |= pa > pb || (pa == pb && sidx[e - 1] >= idx[c]);
                        }
                    }
                }
                if (__syncthreads_or(bad || prm.force_redo)) {
                    if (tid == 0) atomicAdd(prm.redo, 1ull);
#pragma unroll
                    for (int c = 0; c < KPT; ++c) {
                        const uint32_t e = wbase + c * 32 + lane;
                        key[c] = e < count ? kin_map(ksrc[e]) : K(0);  // the source is untouched until the write-out
                        idx[c] = e;
                    }
                    pair_passes(false);
                }
            }
            if (moved || src != SRC_OUT || typed) {
                K *const kd = kout + offs;
                VT *const vd = HV ? vout + offs : nullptr;
                const VT *const vsp = HV ? vs + sv.pad : nullptr;
#pragma unroll
                for (int c = 0; c < KPT; ++c) {
                    const uint32_t e = wbase + c * 32 + lane;
                    if ((!BAL || c < kpt) && e < count) {
                        kd[e] = kout_map(key[c]);
                        if (HV) vd[e] = vsp[idx[c]];
                    }
                }
            }
        }
        __syncthreads();  // staging buffer s, info[s] and red[] are free
        if (tid == 0) {
            fence_proxy_async();
            issue(s, info[16 * NSTAGE]);
            info[16 * NSTAGE] = info[16 * s] + gridDim.x;
        }
    }
}

// ------------------------------------------------------------------ counting local sort
//
// The local sort of a bucket as ONE counting pass instead of
// ceil(bits / 8) LSD passes: a counting sort (histogram -> exclusive prefix -> placement,
// the same three steps as a counting pass) on the CB <= 15 sort bits below the
// entry's top bit (hi_bit: the bits above it are common to the bucket; HRS_LC_NORED=0
// finds the top varying bit with an AND/OR reduction instead), with 2^CB four-bit
// counters packed eight to a word.  2^CB is
// many times the bucket size (<= 4608), so the counted values are nearly distinct; the
// records that tie on them (about one in eight for uniform keys) are put in order by a
// short insertion sort of each tie run, on the remaining sort bits and then the input
// index -- so the result is the stable sort.  The placement slot of a record is
// prefix(word) + counts of the smaller values in its word + the count returned by its
// own counter increment (any order among the ties: the fix-up orders them).
//
// Buckets it does not take go to a hand-off list sorted afterwards by k_local:
//   * at most 8 sort bits (one LSD pass is cheaper);
//   * a counted value held by more than 15 records (four-bit counter overflow: skewed keys);
//   * RECON: more than 19 varying sort bits (the keys are rebuilt from the composites).
// Per record: one shared atomic, two lookups, one composite store and the value gather
// -- about 30 shared-memory wavefronts per 32 records against about 42 for two LSD passes
// (profiles/).
constexpr int LC_SCAN = 256;  // threads that scan the counters
#ifndef HRS_LC_RUNDIV
#define HRS_LC_RUNDIV 3
#endif
// the values of a bucket complete on their own barrier, waited for just before the
// write-out: their load overlaps the count, scan and placement of the bucket
// the top varying sort bit of a bucket is taken from its entry (hi_bit) instead of an
// AND/OR reduction over the bucket's keys (one barrier less per bucket)
#ifndef HRS_LC_NORED
#define HRS_LC_NORED 1
#endif
#ifndef HRS_LC_PL2
#define HRS_LC_PL2 0  // measured slower (spills at 64 registers): c2 local 0.647 + 0.648 -> 0.695 + 0.769 ms
#endif
#ifndef HRS_LC_EARLYK
#define HRS_LC_EARLYK 0  // (measured slower: c2 local 0.646 + 0.659 -> 0.653 + 0.671 ms)
#endif
#ifndef HRS_LC_ALLWAIT
#define HRS_LC_ALLWAIT 1
#endif
#ifndef HRS_LC_VSPLIT
#define HRS_LC_VSPLIT 1
#endif

template <int CB>
struct CntGeom {
    static constexpr int NW = (1 << CB) / 8;      // counter words
    static constexpr int PW = NW / LC_SCAN;       // words per scanning thread
    static_assert(PW >= 1 && PW <= 32 && (PW & (PW - 1)) == 0, "scan geometry");
    // word w lives at t*PW + (k ^ swz(t)) (t = w / PW, k = w % PW): the scanning threads
    // t = 0..31 of a warp reading their k-th words hit 32 different banks
    __device__ __forceinline__ static uint32_t swz(uint32_t t) { return ((t & 31u) * PW / 32u) & (PW - 1u); }
    // = t*PW + (k ^ swz(t)): swz(t) < PW only touches the bits of k
    __device__ __forceinline__ static uint32_t phys(uint32_t w) { return w ^ ((w >> 5) & (PW - 1u)); }
};

// a copy the compiler cannot see through: values recomputed after a barrier are not
// kept live across it (register pressure)
__device__ __forceinline__ uint32_t opaque(uint32_t x) {
    uint32_t y;
    asm volatile("mov.b32 %0, %1;" : "=r"(y) : "r"(x));
    return y;
}

// sum of the eight 4-bit fields of x
__device__ __forceinline__ uint32_t nib_sum(uint32_t x) {
    x = (x & 0x0F0F0F0Fu) + ((x >> 4) & 0x0F0F0F0Fu);
    return (x * 0x01010101u) >> 24;
}

template <typename K, typename V, int THREADS, int KPT, int NSTAGE, int CB, bool RECON>
struct LocalCntSmem {
    static constexpr int W = THREADS / 32;
    static constexpr int CAP = THREADS * KPT;
    using VT = ValT<V>;
    static constexpr bool HV = HasVal<V>::value;
    using G = CntGeom<CB>;
    static constexpr bool VSPLIT = HRS_LC_VSPLIT && HV;  // [NSTAGE + s]: values of stage s
    // EARLYK: the next bucket's keys are loaded while this bucket's values are written out
    // (the key staging buffer holds the composites, read into registers first; RECON only:
    // nothing else reads the key staging buffer in the write-out); [2 NSTAGE]: the
    // composites are consumed (one arrival per warp)
    static constexpr bool EARLYK = HRS_LC_EARLYK && RECON && (VSPLIT || !HV);
    static constexpr size_t off_bar = 0;
    static constexpr size_t off_info = align16(sizeof(uint64_t) * (2 * NSTAGE + 1));
    static constexpr size_t off_red = align16(off_info + sizeof(uint32_t) * 16 * (NSTAGE + 1));
    static constexpr size_t off_wsum = align16(off_red + sizeof(K) * 2 * W);
    static constexpr size_t off_cnt = align16(off_wsum + sizeof(uint32_t) * 16);
    static constexpr size_t off_pref = off_cnt + sizeof(uint32_t) * G::NW;
    // tie runs sorted before the write-out: runs of two or more records (at most CAP / 2),
    // with RECON only runs of three or more (the composite holds every sort bit, pairs are
    // ordered at the write-out), at most RUNCAP of them (more: the bucket is handed off)
    static constexpr int RUNCAP = RECON ? CAP / HRS_LC_RUNDIV : CAP / 2;
    static constexpr size_t off_runs = align16(off_pref + sizeof(uint16_t) * G::NW);
    static constexpr size_t off_comp = align16(off_runs + sizeof(uint32_t) * RUNCAP);
    // RECON: the composites overwrite the key staging buffer (the keys are in registers)
    static constexpr size_t off_kst = align16(off_comp + (RECON ? 0 : sizeof(uint32_t) * CAP));
    static constexpr size_t kst_bytes = align16(sizeof(K) * (CAP + 32 / sizeof(K)));
    static constexpr size_t off_vst = off_kst + NSTAGE * kst_bytes;
    static constexpr size_t vst_bytes = HV ? align16(sizeof(VT) * (CAP + 32 / sizeof(VT))) : 0;
    static constexpr size_t bytes = off_vst + NSTAGE * vst_bytes;
};

template <typename K, typename V, int THREADS, int KPT, int NSTAGE, int MINB, int CB, bool RECON, bool TY>
__global__ void __launch_bounds__(THREADS, MINB) k_local_cnt(LocalParams prm) {
    pdl_wait();
    using L = LocalCntSmem<K, V, THREADS, KPT, NSTAGE, CB, RECON>;
    using G = CntGeom<CB>;
    constexpr int IB = 13;     // index bits of a composite
    constexpr int CBITS = 19;  // sort bits of a composite
    constexpr bool NORED = HRS_LC_NORED;
    static_assert(CBITS <= 24, "a record's register holds the composite's key field below bit 24");
    constexpr uint32_t IMASK = (1u << IB) - 1u;
    constexpr int W = THREADS / 32;
    constexpr int KBITS = 8 * static_cast<int>(sizeof(K));
    constexpr bool HV = HasVal<V>::value;
    using VT = ValT<V>;
    static_assert(THREADS >= LC_SCAN, "the counter scan needs 256 threads");
    static_assert(L::CAP <= (1 << IB), "bucket capacity exceeds the composite index");
    static_assert(!RECON || sizeof(K) == 4, "keys are rebuilt from 32-bit composites only");
    extern __shared__ __align__(16) unsigned char smem[];
    uint64_t *bar = reinterpret_cast<uint64_t *>(smem + L::off_bar);
    uint32_t *info = reinterpret_cast<uint32_t *>(smem + L::off_info);
    K *red = reinterpret_cast<K *>(smem + L::off_red);
    uint32_t *wsum = reinterpret_cast<uint32_t *>(smem + L::off_wsum);
    uint32_t *cnt = reinterpret_cast<uint32_t *>(smem + L::off_cnt);
    uint16_t *pref = reinterpret_cast<uint16_t *>(smem + L::off_pref);
    uint32_t *runs = reinterpret_cast<uint32_t *>(smem + L::off_runs);
    uint32_t *nruns = wsum + 15;  // entries in runs[] (wsum[0 .. LC_SCAN / 32) hold the scan)
    auto kst = [&](int s) { return reinterpret_cast<K *>(smem + L::off_kst + s * L::kst_bytes); };
    auto vst = [&](int s) { return reinterpret_cast<VT *>(smem + L::off_vst + s * L::vst_bytes); };
    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    const uint32_t nent = *prm.count;
    if (blockIdx.x >= nent) return;
    K *__restrict__ kout = static_cast<K *>(prm.keys_out);
    VT *__restrict__ vout = static_cast<VT *>(prm.vals_out);
    const uint64_t pol = policy_evict_first();
    const int begin_bit = prm.begin_bit;

    auto srck = [&](uint32_t code) -> const K * {
        return static_cast<const K *>(code == SRC_IN    ? prm.src_keys[SRC_IN]
                                      : code == SRC_AUX ? prm.src_keys[SRC_AUX]
                                                        : prm.src_keys[SRC_OUT]);
    };
    auto srcv = [&](uint32_t code) -> const VT * {
        return static_cast<const VT *>(code == SRC_IN    ? prm.src_vals[SRC_IN]
                                       : code == SRC_AUX ? prm.src_vals[SRC_AUX]
                                                         : prm.src_vals[SRC_OUT]);
    };
    // info[s]: 0 entry, 1 count, 2 hi_bit, 3 src, 4..5 offs, 6..8 key seg, 9..11 value seg
    // the next entry of the list, fetched while the current bucket is sorted
    LocalEntry *const ahead = reinterpret_cast<LocalEntry *>(info + 16 * NSTAGE + 4);
    // mode bit 0: the keys (and info[s]), bit 1: the values (VSPLIT; else they come with the keys)
    auto issue = [&](int s, uint32_t e, const LocalEntry &en, int mode) {
        uint32_t *in = info + 16 * s;
        if (!(mode & 1)) {  // the values of the entry whose keys were issued earlier
            if constexpr (L::VSPLIT) {
                if (e >= nent) {
                    mbar_arrive_expect_tx(&bar[NSTAGE + s], 0);
                    return;
                }
                Seg sv;
                sv.pad = in[9];
                sv.i0 = static_cast<int32_t>(in[10]);
                sv.i1 = static_cast<int32_t>(in[11]);
                mbar_arrive_expect_tx(&bar[NSTAGE + s], sv.i1 > sv.i0 ? static_cast<uint32_t>(sv.i1 - sv.i0) * static_cast<uint32_t>(sizeof(VT)) : 0u);
                seg_issue(vst(s), srcv(en.src) + en.offs, sv, &bar[NSTAGE + s], pol);
            }
            return;
        }
        in[0] = e;
        if (e >= nent) {
            mbar_arrive_expect_tx(&bar[s], 0);  // completes the phase: the waiters see the end
            if constexpr (L::VSPLIT) if (mode & 2) mbar_arrive_expect_tx(&bar[NSTAGE + s], 0);
            return;
        }
        in[1] = en.count;
        in[2] = en.hi_bit;
        in[3] = en.src;
        in[4] = static_cast<uint32_t>(en.offs);
        in[5] = static_cast<uint32_t>(en.offs >> 32);
        Seg sk, sv;
        const K *kbuf = srck(en.src);
        uint32_t bytes = seg_plan(kbuf + en.offs, en.count, kbuf, kbuf + prm.n, sk);
        in[6] = sk.pad;
        in[7] = static_cast<uint32_t>(sk.i0);
        in[8] = static_cast<uint32_t>(sk.i1);
        uint32_t vbytes = 0;
        if (HV) {
            const VT *vbuf = srcv(en.src);
            vbytes = seg_plan(vbuf + en.offs, en.count, vbuf, vbuf + prm.n, sv);
            in[9] = sv.pad;
            in[10] = static_cast<uint32_t>(sv.i0);
            in[11] = static_cast<uint32_t>(sv.i1);
        }
        mbar_arrive_expect_tx(&bar[s], L::VSPLIT ? bytes : bytes + vbytes);
        seg_issue(kst(s), kbuf + en.offs, sk, &bar[s], pol);
        if (L::VSPLIT && !(mode & 2)) return;
        if constexpr (L::VSPLIT) mbar_arrive_expect_tx(&bar[NSTAGE + s], vbytes);
        if (HV) seg_issue(vst(s), srcv(en.src) + en.offs, sv, &bar[L::VSPLIT ? NSTAGE + s : s], pol);
    };
    auto hand_off = [&](uint64_t offs, uint32_t count, int hi_bit, uint32_t src) {
        const uint32_t slot = atomicAdd(prm.fb_count, 1u);
        if (slot < prm.fb_cap) {
            LocalEntry en;
            en.offs = offs;
            en.count = count;
            en.hi_bit = static_cast<uint16_t>(hi_bit);
            en.src = static_cast<uint16_t>(src);
            prm.fb_list[slot] = en;
        }
    };
    for (int i = tid; i < G::NW; i += THREADS) cnt[i] = 0;  // cleared again after every bucket
    if (tid == 0) {
        for (int s = 0; s < 2 * NSTAGE; ++s) mbar_init(&bar[s], 1);
        mbar_init(&bar[2 * NSTAGE], W);
        mbar_fence_init();
        for (int s = 0; s < NSTAGE; ++s) {
            const uint32_t e = blockIdx.x + s * gridDim.x;
            LocalEntry en{};
            if (e < nent) en = prm.list[e];
            issue(s, e, en, 3);
        }
        info[16 * NSTAGE] = blockIdx.x + NSTAGE * gridDim.x;  // next entry to issue
        *nruns = 0;
    }
    __syncthreads();
    bool keys_early = false;  // (tid 0) the next entry's keys are already in flight
    uint32_t cf_par = 0;      // (tid 0) phase of the composites-consumed barrier

    for (uint32_t it = 0;; ++it) {
        const int s = static_cast<int>(it % NSTAGE);
        const uint32_t par = (it / NSTAGE) & 1u;
        const uint32_t *in = info + 16 * s;
        // the bulk copies of the keys (the producer wrote info[s] before its arrive: the wait
        // acquires it).  ALLWAIT: every thread waits on the barrier itself (no CTA barrier);
        // else one warp waits and a CTA barrier passes both on to the other warps
        if (HRS_LC_ALLWAIT || warp == 0) mbar_wait(&bar[s], par);
        if (!HRS_LC_ALLWAIT) __syncthreads();
        const uint32_t e_id = in[0];
        if (e_id >= nent) break;
        if (tid == 0 && info[16 * NSTAGE] < nent) cp_async16(ahead, prm.list + info[16 * NSTAGE]);
        const uint32_t count = in[1];
        const int hi_bit = static_cast<int>(in[2]);
        const uint32_t src = in[3];
        // signed / float keys (hrs_sort_typed): keys read from the input are mapped to their
        // order-preserving image, every key this kernel writes is final and mapped back
        const bool typed = TY && prm.kind != 0;
        const bool mapin = typed && src == SRC_IN;
        auto kin_map = [&](K x) -> K { return mapin ? key_map(x, prm.kind, false) : x; };
        auto kout_map = [&](K x) -> K { return typed ? key_map(x, prm.kind, true) : x; };
        // a staged key copied to the output: the original if it came from the input
        auto kout_raw = [&](K x) -> K { return (typed && !mapin) ? key_map(x, prm.kind, true) : x; };
        const uint64_t offs = static_cast<uint64_t>(in[4]) | (static_cast<uint64_t>(in[5]) << 32);
        Seg sk, sv;
        sk.pad = in[6];
        sk.i0 = static_cast<int32_t>(in[7]);
        sk.i1 = static_cast<int32_t>(in[8]);
        sv.pad = in[9];
        sv.i0 = static_cast<int32_t>(in[10]);
        sv.i1 = static_cast<int32_t>(in[11]);
        const K *ksrc = srck(src) + offs;
        const VT *vsrc = HV ? srcv(src) + offs : nullptr;
        K *ks = kst(s);
        VT *vs = HV ? vst(s) : nullptr;
        // VSPLIT: every thread waits for the values itself before it reads them
        auto vwait = [&]() {
            if constexpr (L::VSPLIT) mbar_wait(&bar[NSTAGE + s], par);
        };
        // elements the bulk copy did not cover (entries at the ends of a buffer): into
        // shared memory before anything is written (the entry may be sorted in place)
        if (!seg_full(sk, count) || (HV && !seg_full(sv, count))) {
            seg_fill_edges<K, THREADS>(ks, ksrc, sk, count);
            if (HV) seg_fill_edges<VT, THREADS>(vs, vsrc, sv, count);
            __syncthreads();
        }
        const K *const ksp = ks + sk.pad;
        K key[KPT];
        K a = ~K(0), o = K(0);
#pragma unroll
        for (int c = 0; c < KPT; ++c) {
            const uint32_t e = c * THREADS + tid;
            key[c] = kin_map(ksp[e < count ? e : 0u]);  // past the end: a copy of key 0 (neutral for and/or)
            if constexpr (!NORED) {
                a &= key[c];
                o |= key[c];
            }
        }
        // thi: the top sort bit that varies across the bucket (counted bits [thi - CB, thi)).
        // NORED: the entry's hi_bit -- every key bit at or above it is common to the bucket
        // (its partitioned digits; a merged group's hi_bit is the top bit in which its digits
        // differ) and the next bit below varies in practice for buckets of > 2048 records;
        // were it constant, the counted values would tie more (overflow: hand-off), never a
        // different result.  Saves the AND/OR reduction and its barrier.
        K aa, diff;
        int thi = 0;
        bool nosort;
        if constexpr (NORED) {
            thi = hi_bit;
            aa = key[0];  // (bits >= thi: common to the bucket)
            diff = K(0);
            nosort = false;
        } else {
            a = warp_and(a);
            o = warp_or(o);
            if (lane == 0) {
                red[warp] = a;
                red[W + warp] = o;
            }
            __syncthreads();  // B1: red[], filled edges
            aa = ~K(0);
            K oo = K(0);
#pragma unroll
            for (int w = 0; w < W; ++w) {
                aa &= red[w];
                oo |= red[W + w];
            }
            diff = aa ^ oo;
            const K rmask = (hi_bit >= KBITS ? ~K(0) : ((K(1) << hi_bit) - 1)) & ~((K(1) << begin_bit) - 1);
            const K dv = diff & rmask;  // sort bits that vary across the bucket
            if (dv != 0) thi = KBITS - (sizeof(K) == 8 ? __clzll(static_cast<long long>(dv)) : __clz(static_cast<int>(dv)));
            nosort = dv == 0;
        }
        const int clo = max(begin_bit, thi - CBITS);  // composite: key bits [clo, thi)
        const int flo = max(clo, thi - CB);           // counted: key bits [flo, thi)
        bool take = !nosort && thi - begin_bit > 8;
        if (RECON) take = take && begin_bit == 0 && clo == 0 && (thi >= KBITS || (diff >> thi) == 0);
        K *const kd = kout + offs;
        VT *const vd = HV ? vout + offs : nullptr;
        const VT *const vsp = HV ? vs + sv.pad : nullptr;
        if (nosort) {
            // every record has the same sort bits: the stable order is the input order
            if (src != SRC_OUT || typed) {
                vwait();
#pragma unroll
                for (int c = 0; c < KPT; ++c) {
                    const uint32_t e = c * THREADS + tid;
                    if (e < count) {
                        kd[e] = kout_map(key[c]);
                        if (HV) vd[e] = vsp[e];
                    }
                }
            }
        } else if (!take) {
            if (tid == 0) hand_off(offs, count, hi_bit, src);
        } else {
            const int FS = IB + (flo - clo);  // composite >> FS = counted value
            const uint32_t cmask = (1u << (thi - clo)) - 1u;
            // the composites' buffer (RECON: the key staging buffer, whose keys are now in
            // registers); low: key bits below the composite decide ties
            uint32_t *const comp = RECON ? reinterpret_cast<uint32_t *>(ks) : reinterpret_cast<uint32_t *>(smem + L::off_comp);
            const bool low = clo > begin_bit;
            constexpr uint32_t SENT = 0xFFFFFFFFu;  // no composite (index bits 8191 > CAP)
            static_assert(L::CAP < (1 << IB) - 1, "SENT is not a composite");
            // one register per record from the count to the placement: the composite's key
            // field (<= CBITS bits) and the record's rank among its ties (bits 24..27); the
            // composite, counted value, word and nibble are recomputed from them (registers:
            // five CTAs per SM where the shared memory allows)
            const int VSH = flo - clo;  // key field >> VSH = counted value
            uint32_t rec[KPT];
#pragma unroll
            for (int c = 0; c < KPT; ++c) {
                const uint32_t e = c * THREADS + tid;
                const uint32_t kf = static_cast<uint32_t>(key[c] >> clo) & cmask;
                rec[c] = kf;  // (past the end: a valid counter word for the placement's loads)
                if (e < count) {
                    if constexpr (RECON && !NORED) comp[e] = SENT;  // (tie pairs swap into their first slot)
                    const uint32_t v = kf >> VSH;
                    const uint32_t ph = G::phys(v >> 3), sh = (v & 7u) * 4u;
                    const uint32_t on = (atomicAdd(&cnt[ph], 1u << sh) >> sh) & 15u;
                    rec[c] = kf | (on << 24);
                }
            }
            __syncthreads();  // B2 (counts complete)
            if constexpr (RECON && NORED) {
                // (after B2: without B1 another thread may read its key from the staging buffer,
                // which the composites overwrite, until then)
#pragma unroll
                for (int c = 0; c < KPT; ++c) {
                    const uint32_t e = c * THREADS + tid;
                    if (e < count) comp[e] = SENT;  // (tie pairs swap into their first slot)
                }
            }
            {
                // exclusive prefix of the word totals: 256 threads own PW consecutive words.
                // A counter that passed 15 wrapped (-16, +1 carried into its neighbour or
                // lost): the nibble total then falls short of count, checked after B3.
                uint32_t ws[G::PW];
                uint32_t tsum = 0, incl = 0;
                const uint32_t sw = G::swz(static_cast<uint32_t>(tid));
                if (tid < LC_SCAN) {
#pragma unroll
                    for (int k = 0; k < G::PW; ++k) {
                        ws[k] = nib_sum(cnt[tid * G::PW + (k ^ sw)]);
                        tsum += ws[k];
                    }
                    incl = tsum;
#pragma unroll
                    for (int d = 1; d < 32; d <<= 1) {
                        const uint32_t y = __shfl_up_sync(0xffffffffu, incl, d);
                        if (lane >= d) incl += y;
                    }
                    if (lane == 31) wsum[warp] = incl;
                }
                __syncthreads();  // B3
                uint32_t total = 0;
#pragma unroll
                for (int w = 0; w < LC_SCAN / 32; ++w) total += wsum[w];
                if (total != count) {  // four-bit counter overflow: k_local takes the bucket
                    for (int i = tid; i < G::NW; i += THREADS) cnt[i] = 0;
                    if (tid == 0) hand_off(offs, count, hi_bit, src);
                    goto next_entry;
                }
                if (tid < LC_SCAN) {
                    uint32_t base = incl - tsum;
#pragma unroll
                    for (int w = 0; w < LC_SCAN / 32; ++w) base += w < warp ? wsum[w] : 0u;
#pragma unroll
                    for (int k = 0; k < G::PW; ++k) {
                        pref[tid * G::PW + (k ^ sw)] = static_cast<uint16_t>(base);
                        base += ws[k];
                    }
                }
                __syncthreads();  // B4
                // slot = prefix of the word + counts of the smaller values in the word + the
                // record's own rank among the ties.  The record that counted first (on == 0)
                // of a value held by r > 1 records owns that tie run.  When the composite holds
                // every sort bit (!low) a pair is ordered without the list: here (RECON, atomic
                // exchange into its first slot) or at the write-out (min / max of the two
                // neighbours); longer runs, and every run when key bits below the composite
                // decide (low), go to a list that the whole CTA sorts before the write-out
                const uint32_t r0 = low ? 2u : 3u;
                // PL2: every record's slot and tie count first (loads of all records in flight
                // together, no branches), then the stores
                [[maybe_unused]] uint32_t sr[HRS_LC_PL2 ? KPT : 1];
                if constexpr (HRS_LC_PL2) {
#pragma unroll
                    for (int c = 0; c < KPT; ++c) {
                        const uint32_t kf = rec[c] & 0xFFFFFFu, on = rec[c] >> 24;
                        const uint32_t v = kf >> VSH;
                        const uint32_t ph = G::phys(v >> 3), sh = (v & 7u) * 4u;
                        const uint32_t w = cnt[ph];
                        const uint32_t slot = pref[ph] + nib_sum(w & ((1u << sh) - 1u)) + on;
                        sr[c] = slot | (((w >> sh) & 15u) << 16);
                    }
                }
#pragma unroll
                for (int c = 0; c < KPT; ++c) {
                    const uint32_t e = c * THREADS + tid;
                    if (e < count) {
                        const uint32_t kf = rec[c] & 0xFFFFFFu, on = rec[c] >> 24;
                        const uint32_t cvc = (kf << IB) | e;
                        uint32_t slot, r;
                        if constexpr (HRS_LC_PL2) {
                            slot = sr[c] & 0xFFFFu;
                            r = sr[c] >> 16;
                        } else {
                            const uint32_t v = kf >> VSH;
                            const uint32_t ph = G::phys(v >> 3), sh = (v & 7u) * 4u;
                            const uint32_t w = cnt[ph];
                            slot = pref[ph] + nib_sum(w & ((1u << sh) - 1u)) + on;
                            r = (w >> sh) & 15u;
                        }
                        if (RECON && r == 2u) {
                            // (RECON: the composite holds every sort bit) a tie pair orders
                            // itself: the second record to arrive swaps its composite in and
                            // writes the two in order (the slots start as SENT)
                            const uint32_t b0 = slot - on, old = atomicExch(&comp[b0], cvc);
                            if (old != SENT) {
                                comp[b0] = min(old, cvc);
                                comp[b0 + 1] = max(old, cvc);
                            }
                        } else {
                            comp[slot] = cvc;
                        }
                        if (on == 0 && r >= r0) {
                            const uint32_t q = atomicAdd(nruns, 1u);
                            if (q < L::RUNCAP) runs[q] = slot | (r << 16);
                        }
                    }
                }
                __syncthreads();  // B5
                for (int i = tid; i < G::NW; i += THREADS) cnt[i] = 0;
                const uint32_t nr = *nruns;
                if (nr > L::RUNCAP) {  // more tie runs than the list holds: k_local takes the bucket
                    if (tid == 0) hand_off(offs, count, hi_bit, src);
                    goto next_entry;
                }
                if (nr) {
                    // tie runs (equal counted value, at most 15 records): insertion sort by the
                    // rest of the composite, then the key bits below it, then the index
                    const int lb = clo - begin_bit;
                    const K lmask = lb >= KBITS ? ~K(0) : ((K(1) << lb) - 1);
                    auto less = [&](uint32_t x, uint32_t y) -> bool {
                        if ((x >> IB) != (y >> IB)) return x < y;
                        if (low) {
                            const K lx = (kin_map(ksp[x & IMASK]) >> begin_bit) & lmask,
                                    ly = (kin_map(ksp[y & IMASK]) >> begin_bit) & lmask;
                            if (lx != ly) return lx < ly;
                        }
                        return x < y;
                    };
                    for (uint32_t q = tid; q < nr; q += THREADS) {
                        const uint32_t rn = runs[q];
                        uint32_t *rb = comp + (rn & 0xFFFFu);
                        const uint32_t r = rn >> 16;
                        for (uint32_t i = 1; i < r; ++i) {
                            const uint32_t x = rb[i];
                            int j = static_cast<int>(i) - 1;
                            while (j >= 0) {
                                const uint32_t y = rb[j];
                                if (!less(x, y)) break;
                                rb[j + 1] = y;
                                --j;
                            }
                            rb[j + 1] = x;
                        }
                    }
                    __syncthreads();  // B6
                }
                // write-out: RECON rebuilds the key from the bits above thi (common to
                // the bucket) and the composite's sort field; otherwise it is gathered
                const K khigh = thi >= KBITS ? K(0) : (aa & ~((K(1) << thi) - 1));
                const uint32_t fs2 = opaque(static_cast<uint32_t>(FS));
                vwait();
                if constexpr (L::EARLYK) {
                    // composites into registers, the key staging buffer is free: the next
                    // entry's keys load while the values are gathered and written
                    uint32_t xs[KPT];
#pragma unroll
                    for (int c = 0; c < KPT; ++c) {
                        const uint32_t e = c * THREADS + tid;
                        xs[c] = e < count ? comp[e] : 0u;
                    }
                    __syncwarp();
                    if (lane == 0) mbar_arrive(&bar[2 * NSTAGE]);
                    if (tid == 0) {
                        mbar_wait(&bar[2 * NSTAGE], cf_par);
                        cf_par ^= 1u;
                        fence_proxy_async();
                        cp_async_wait_all();
                        issue(s, info[16 * NSTAGE], *ahead, 1);
                        keys_early = true;
                    }
#pragma unroll
                    for (int c = 0; c < KPT; ++c) {
                        const uint32_t e = c * THREADS + tid;
                        if (e < count) {
                            const uint32_t x = xs[c];
                            kd[e] = kout_map(khigh | static_cast<K>(x >> IB));
                            if (HV) vd[e] = vsp[x & IMASK];
                        }
                    }
                    goto next_entry;
                }
#pragma unroll
                for (int c = 0; c < KPT; ++c) {
                    const uint32_t e = c * THREADS + tid;
                    if (e < count) {
                        uint32_t x = comp[e];
                        if (!RECON && !low) {
                            // first of a run: the smaller of itself and its successor; last: the
                            // larger of its predecessor and itself; inside a (sorted) longer run
                            // or alone: itself
                            const uint32_t xp = comp[e > 0 ? e - 1 : 0], xn = comp[e + 1 < L::CAP ? e + 1 : e];
                            const uint32_t v = x >> fs2;
                            const bool sp = e > 0 && (xp >> fs2) == v, sn = e + 1 < count && (xn >> fs2) == v;
                            if (sn && !sp) x = min(x, xn);
                            if (sp && !sn) x = max(x, xp);
                        }
                        const uint32_t ix = x & IMASK;
                        kd[e] = RECON ? kout_map(khigh | static_cast<K>(x >> IB)) : kout_raw(ksp[ix]);
                        if (HV) vd[e] = vsp[ix];
                    }
                }
            }
        }
    next_entry:
        __syncthreads();  // staging buffer s, info[s], red[], comp, the run list are free
        if (tid == 0) {
            *nruns = 0;
            vwait();  // (a bucket handed off never waited: the phase completes before the re-arm)
            fence_proxy_async();
            cp_async_wait_all();
            issue(s, info[16 * NSTAGE], *ahead, keys_early ? 2 : 3);
            info[16 * NSTAGE] += gridDim.x;
            keys_early = false;
        }
    }
}

}  // namespace hrs
