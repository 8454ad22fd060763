/*
 * hrs.h -- C ABI of the B200-native (sm_100a) hybrid radix sort.
 *
 * Method: Stehle & Jacobsen, "A Memory Bandwidth-Efficient Hybrid Radix Sort on
 * GPUs", SIGMOD'17 (arXiv 1611.01137).  PAPER.md line citations are P:<line>.
 *   - MSD radix sort with 8-bit digits (d = 8): every bucket larger than
 *     the local-sort threshold ∂ˆ is partitioned by a counting sort -- histogram,
 *     exclusive prefix sum into sub-bucket offsets, scatter -- and
 *     every bucket of at most ∂ˆ records is finished by an on-chip local sort
 *     (R1/R2 P:805-808).  Tiny neighbouring sub-buckets are merged while
 *     their total is below ∂ (R3 P:809-811).
 *   - Departure from the paper: every pass is STABLE, so
 *     the output is the unique stable sort and is bit-identical run to run.
 *
 * Semantics of every hrs_sort_* call:
 *   With W = end_bit - begin_bit and sk(x) = (x >> begin_bit) mod 2^W, the output
 *   is keys_in[pi(i)] (and vals_in[pi(i)]) for the unique permutation pi such that
 *   (sk(keys_in[pi(i)]), pi(i)) is strictly increasing: ties keep input order.
 *   Key bits outside [begin_bit, end_bit) are carried unchanged.  n == 0 is a no-op;
 *   begin_bit == end_bit is a stable copy.
 *
 * Conventions
 *   Memory:    every data pointer (keys, values, temp, d_hist, d_offsets) is a CUDA
 *              device pointer owned by the caller, naturally aligned for its type
 *              (temp: 256 bytes).  The library never allocates, frees or retains
 *              device memory.  Inputs are const; keys_in/keys_out/vals_in/vals_out/
 *              temp must not overlap (HRS_ERROR_ALIASING).
 *   Temp:      two-phase protocol: with d_temp == NULL the call stores the required
 *              size in *temp_bytes, enqueues nothing and returns HRS_SUCCESS.
 *              Otherwise *temp_bytes is the size of d_temp.
 *   Streams:   work is enqueued on `stream` (NULL = legacy default stream) and the
 *              call returns without synchronising (no device->host reads inside the
 *              sort, so calls can be captured in CUDA graphs).  hrs_get_stats is the
 *              only entry point that synchronises its stream.
 *   Errors:    argument errors are returned synchronously; a CUDA launch error maps
 *              to HRS_ERROR_CUDA with the cudaError_t in hrs_last_cuda_error()
 *              (thread-local).  Device faults surface at the caller's next sync.
 *              No C++ exception crosses this ABI.
 *   Devices:   the library contains sm_100a code only; on any other device the
 *              calls fail with HRS_ERROR_NO_DEVICE.  There is no CPU fallback.
 *   Graphs:    sorts of at most 2^22 records are launch-bound: from the second call
 *              with identical arguments (every pointer included) the library replays
 *              a CUDA graph of its launch sequence, captured on a private stream, with
 *              one cudaGraphLaunch into `stream` (not while `stream` is itself being
 *              captured; environment HRS_GRAPHS=0 disables it).
 *   Threads:   stateless apart from the thread-local last error, per-device
 *              launch-configuration caches and the graph cache (mutex-protected);
 *              concurrent calls on different streams with different temp buffers
 *              are safe.
 *   Limits:    n <= HRS_MAX_ITEMS.
 */
#ifndef HRS_H_
#define HRS_H_

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif
#if defined(__GNUC__)
#pragma GCC visibility push(default) /* the library is built with -fvisibility=hidden */
#endif

#define HRS_MAX_ITEMS 0xFFFFFFFFull /* counts are 32-bit inside the kernels ("easily adjusted") */

typedef struct CUstream_st *hrs_stream_t; /* identical to cudaStream_t */

typedef enum {
    HRS_SUCCESS = 0,
    HRS_ERROR_INVALID_VALUE = 1,  /* NULL pointer with n > 0, NULL temp_bytes, misaligned pointer, bad tuning */
    HRS_ERROR_INVALID_BITS = 2,   /* not 0 <= begin_bit <= end_bit <= key bits (digit range for building blocks) */
    HRS_ERROR_ALIASING = 3,       /* any overlap among the data buffers and temp */
    HRS_ERROR_TEMP_TOO_SMALL = 4, /* *temp_bytes smaller than required */
    HRS_ERROR_TOO_LARGE = 5,      /* n > HRS_MAX_ITEMS */
    HRS_ERROR_NO_DEVICE = 6,      /* current device is not an sm_100 GPU */
    HRS_ERROR_CUDA = 7            /* a CUDA call failed; see hrs_last_cuda_error() */
} hrs_status;

/* Tuning override (tests and ablations).  0 in a field = the default for the
 * key/value types.  Thresholds change performance, never results.
 *   local_threshold  ∂ˆ  buckets with <= ∂ˆ records are local-sorted (1 .. hrs_max_local_threshold)
 *   merge_threshold  ∂   neighbouring sub-buckets merge while their total < ∂ (1 .. ∂ˆ; 1 = no merging)
 *   keys_per_tile    KPB records per tile ("key block") (1 .. hrs_max_keys_per_tile)
 *   local_classes    0 = size classes [1,128], (128,256], ...; 1 = a single
 *                    local-sort configuration for every bucket (the ablation of Figs 11-14)
 *   flags            HRS_FLAG_* test switches (0 in production).  HRS_FLAG_FORCE_REDO makes
 *                    every stability check of the fast rank fail, so the scatter and the
 *                    local sorts always take their stable-by-construction redo path (the
 *                    fast rank takes the lane order of returning shared-memory atomics as
 *                    the in-warp order, which PTX does not guarantee; the checks catch a
 *                    device that reorders, and this flag is how tests exercise the redo
 *                    code).  The environment variable HRS_FORCE_REDO=1, read once when the
 *                    library loads, ORs it into every call.  Results are identical either
 *                    way; only the time changes. */
typedef struct {
    uint32_t local_threshold;
    uint32_t merge_threshold;
    uint32_t keys_per_tile;
    uint32_t local_classes;
    uint32_t flags;
} hrs_tuning;
#define HRS_FLAG_FORCE_REDO 1u

#define HRS_MAX_PASSES 8
#define HRS_NUM_CLASSES 8

/* Observability block kept inside temp and filled on the device during a sort. */
typedef struct {
    uint64_t n;
    uint32_t key_bytes, value_bytes;
    uint32_t counting_passes;                  /* counting-sort passes executed */
    uint32_t overflow;                         /* non-zero: an internal table bound was exceeded (bug) */
    uint64_t recs_in_pass[HRS_MAX_PASSES];     /* records in buckets partitioned by pass p+1 */
    uint64_t tiles_in_pass[HRS_MAX_PASSES];    /* tiles (key blocks) of pass p+1 */
    uint64_t buckets_in_pass[HRS_MAX_PASSES];  /* buckets partitioned by pass p+1 */
    uint64_t local_buckets;                    /* local-sort entries (after merging) */
    uint64_t local_recs;                       /* records finished by a local sort */
    uint64_t merged_groups;                    /* local entries made of >= 2 merged sub-buckets */
    uint64_t local_in_class[HRS_NUM_CLASSES];  /* local entries per size class */
    uint64_t bytes_min;                        /* sum_p [R_p K + (R_p - S_p) 2(K+V)] + R_L 2(K+V) */
    uint64_t redo_blocks;                      /* tiles / buckets redone with the stable-by-construction rank
                                                  (0 unless a stability check failed or HRS_FLAG_FORCE_REDO) */
    uint64_t skipped_recs_in_pass[HRS_MAX_PASSES]; /* S_p: records of buckets whose digit p is constant and that
                                                  never moved: their scatter is skipped (reading #22) */
} hrs_stats;

/* ---- full sorts; arguments: temp, size, keys in/out, [values in/out], n, bit range, stream ---- */
hrs_status hrs_sort_keys_u32(void *d_temp, size_t *temp_bytes, const uint32_t *keys_in, uint32_t *keys_out,
                             uint64_t n, int begin_bit, int end_bit, hrs_stream_t stream);
hrs_status hrs_sort_keys_u64(void *d_temp, size_t *temp_bytes, const uint64_t *keys_in, uint64_t *keys_out,
                             uint64_t n, int begin_bit, int end_bit, hrs_stream_t stream);
hrs_status hrs_sort_pairs_u32_u32(void *d_temp, size_t *temp_bytes, const uint32_t *keys_in, uint32_t *keys_out,
                                  const uint32_t *vals_in, uint32_t *vals_out, uint64_t n, int begin_bit,
                                  int end_bit, hrs_stream_t stream);
hrs_status hrs_sort_pairs_u32_u64(void *d_temp, size_t *temp_bytes, const uint32_t *keys_in, uint32_t *keys_out,
                                  const uint64_t *vals_in, uint64_t *vals_out, uint64_t n, int begin_bit,
                                  int end_bit, hrs_stream_t stream);
hrs_status hrs_sort_pairs_u64_u32(void *d_temp, size_t *temp_bytes, const uint64_t *keys_in, uint64_t *keys_out,
                                  const uint32_t *vals_in, uint32_t *vals_out, uint64_t n, int begin_bit,
                                  int end_bit, hrs_stream_t stream);
hrs_status hrs_sort_pairs_u64_u64(void *d_temp, size_t *temp_bytes, const uint64_t *keys_in, uint64_t *keys_out,
                                  const uint64_t *vals_in, uint64_t *vals_out, uint64_t n, int begin_bit,
                                  int end_bit, hrs_stream_t stream);

/* Generic form behind the typed entry points.  key_bytes in {4, 8}; value_bytes in
 * {0, 4, 8} (0: vals_in/vals_out ignored, may be NULL); tuning may be NULL. */
hrs_status hrs_sort_ex(void *d_temp, size_t *temp_bytes, const void *keys_in, void *keys_out,
                       const void *vals_in, void *vals_out, uint64_t n, int key_bytes, int value_bytes,
                       int begin_bit, int end_bit, const hrs_tuning *tuning, hrs_stream_t stream);

/* The same stable sort for an input that is ALREADY GROUPED by its first (most
 * significant) digit: the digit of bits [max(begin_bit, end_bit - 8), end_bit), the first
 * digit of the plan, with the records of digit value 0 first, then 1, ... --
 * e.g. what a partition pass on that digit (hrs_partition_pass) or the bucket-major
 * exchange of the distributed sort produces.  d_first_digit_hist (device, 2^width uint64)
 * holds the number of records of every digit value; it must sum to n.  The library takes
 * the first counting pass as done (its histogram, exclusive prefix and sub-bucket
 * classification, run from d_first_digit_hist; nothing is moved) and
 * continues at the second digit, so the sort reads and writes every record once less.
 * Output, temp size, layout, ownership, async behaviour and errors as hrs_sort_ex
 * (HRS_ERROR_INVALID_VALUE if d_first_digit_hist is NULL for a non-trivial sort).  The
 * grouping is a precondition, not checked: an input that is not grouped, or a histogram
 * that does not describe it, gives an unspecified permutation of the input. */
hrs_status hrs_sort_grouped(void *d_temp, size_t *temp_bytes, const void *keys_in, void *keys_out,
                            const void *vals_in, void *vals_out, uint64_t n, int key_bytes, int value_bytes,
                            int begin_bit, int end_bit, const uint64_t *d_first_digit_hist, const hrs_tuning *tuning,
                            hrs_stream_t stream);

/* Copies the stats block of the last sort that used d_temp to *out.  Synchronises
 * `stream`; call it outside any timed region. */
hrs_status hrs_get_stats(const void *d_temp, hrs_stats *out, hrs_stream_t stream);

/* Largest accepted local_threshold / keys_per_tile for the key/value widths. */
uint32_t hrs_max_local_threshold(int key_bytes, int value_bytes);
uint32_t hrs_max_keys_per_tile(int key_bytes, int value_bytes);
/* Default tuning for the key/value widths (written to *out). */
hrs_status hrs_default_tuning(int key_bytes, int value_bytes, hrs_tuning *out);
/* Capacity (largest size) of local-sort size class c, 0 <= c < HRS_NUM_CLASSES (0 for c out
 * of range): a bucket of s records goes to the smallest class whose capacity is >= s
 * (hrs_stats.local_in_class counts entries per class).  P:562-566 gives the classes
 * [1,128], (128,256], (256,512], ... as an example; this build uses powers of two up to
 * 4096, then 4608 and 8192 (reading #20: uniform 2^28 inputs leave buckets of
 * 4096 +- 200 records after two passes). */
uint32_t hrs_class_capacity(int c);

/* ---- signed and floating-point keys (the paper's order-preserving
 * bijections) ----
 * Stable sort of n keys of `kind` by their whole value (no bit range), values moved along:
 *   HRS_KEY_UINT:  unsigned (as hrs_sort_ex over [0, 8 * key_bytes));
 *   HRS_KEY_INT:   two's-complement signed;
 *   HRS_KEY_FLOAT: IEEE-754 binary32 (key_bytes 4) / binary64 (8) in the total order
 *                  -NaN < -inf < ... < -0.0 < +0.0 < ... < +inf < +NaN (NaNs of one sign
 *                  ordered by their bit patterns: larger payload further out).
 * Layout, ownership, async behaviour and errors as hrs_sort_ex; temp as hrs_sort_ex for
 * unsigned keys of the same width.  The bijection (ints: flip the sign bit; floats: flip
 * every bit of a negative key, the sign bit of a positive one) is fused into the sort as
 * P:914-918 describes: a key read from the input is mapped where it is read (the first
 * histogram and scatter, the local sorts of buckets that never moved), and mapped back
 * where it is written for the last time (the last counting pass, the local sorts). */
typedef enum { HRS_KEY_UINT = 0, HRS_KEY_INT = 1, HRS_KEY_FLOAT = 2 } hrs_key_kind;
hrs_status hrs_sort_typed(void *d_temp, size_t *temp_bytes, const void *keys_in, void *keys_out,
                          const void *vals_in, void *vals_out, uint64_t n, int key_bytes, int value_bytes,
                          hrs_key_kind kind, hrs_stream_t stream);

/* ---- records stored interleaved (array of structs) ----
 * Record i is key_bytes + value_bytes bytes at records_in + i * (key_bytes + value_bytes),
 * its key at byte offset key_offset (0: key first, value_bytes: value first), both parts
 * little-endian; records are 4-byte aligned.  The records are decomposed into a key array
 * and a value array (one pass at memory bandwidth; the key of a signed / float kind goes
 * through the order-preserving bijection of hrs_sort_typed on the way), sorted
 * as pairs (hrs_sort_ex; stable), and recomposed into records_out (the inverse bijection
 * fused into that pass).  kind HRS_KEY_UINT sorts by key bits [begin_bit, end_bit); the
 * other kinds by the whole key (begin_bit = 0, end_bit = 8 * key_bytes, else
 * HRS_ERROR_INVALID_BITS).  Temp = 2 n (key_bytes + value_bytes) + the pair sort's temp
 * (two-phase size query); records_in, records_out and temp must not overlap.  Otherwise
 * as hrs_sort_ex. */
hrs_status hrs_sort_records(void *d_temp, size_t *temp_bytes, const void *records_in, void *records_out, uint64_t n,
                            int key_bytes, int value_bytes, int key_offset, int begin_bit, int end_bit,
                            hrs_key_kind kind, hrs_stream_t stream);

/* ---- building blocks (kernel-level tests, the distributed driver) ---- */

/* Histogram of digit bits [lo_bit, hi_bit) (1 <= hi_bit - lo_bit <= 8) over all n keys:
 * step (1) of a counting sort.  d_hist receives 2^(hi-lo) uint64 counts. */
hrs_status hrs_digit_histogram(void *d_temp, size_t *temp_bytes, const void *keys, uint64_t n, int key_bytes,
                               int lo_bit, int hi_bit, uint64_t *d_hist, hrs_stream_t stream);

/* One STABLE counting-sort pass of the whole input on digit bits [lo_bit, hi_bit):
 * histogram, exclusive prefix sum, scatter.  d_offsets receives the
 * 2^(hi-lo) + 1 uint64 bucket starts (the last entry is n).  d_offsets may be NULL. */
hrs_status hrs_partition_pass(void *d_temp, size_t *temp_bytes, const void *keys_in, void *keys_out,
                              const void *vals_in, void *vals_out, uint64_t n, int key_bytes, int value_bytes,
                              int lo_bit, int hi_bit, uint64_t *d_offsets, hrs_stream_t stream);

/* The same stable counting pass, with every digit's run written to its own window: the
 * records of digit d go, in input order, to key window w = dst_offsets[d] >> 48 at element
 * offset dst_offsets[d] & (2^48 - 1) (values likewise, to value window w).  dst_offsets,
 * key_windows and value_windows are HOST arrays (2^(hi-lo) offsets; nwindows <= 64 device
 * addresses each, naturally aligned), copied into d_temp during the call (the call
 * synchronises `stream` once for that copy).  A window may be another GPU's memory mapped
 * into this process (CUDA IPC / symmetric memory over NVLink): this is the fused exchange of
 * the partition scatter stores every bucket run straight into the
 * receiving GPU's buffer, with no local partition buffer and no separate all-to-all.  The
 * runs must not overlap each other or the input; the caller synchronises with the
 * receivers.  Temp size: two-phase query as usual (larger than hrs_partition_pass's). */
hrs_status hrs_partition_pass_to(void *d_temp, size_t *temp_bytes, const void *keys_in, const void *vals_in,
                                 uint64_t n, int key_bytes, int value_bytes, int lo_bit, int hi_bit,
                                 const uint64_t *dst_offsets, int nwindows, const uint64_t *key_windows,
                                 const uint64_t *value_windows, hrs_stream_t stream);

/* Copies npieces pieces of elem_bytes-wide elements (4 or 8) from src to dst (device):
 * `pieces` is a HOST array of npieces x {src_offset, dst_offset, count} uint64, in
 * elements, read during the call (it travels in kernel parameters, 256 pieces per
 * launch; no device memory is needed for it).  The pieces must not overlap in dst, and
 * src and dst must not overlap.  The distributed sort's placement of a rank's own pieces
 * in the bucket-major exchange (the pieces of every first-digit
 * bucket from every source, in source order). */
hrs_status hrs_copy_pieces(void *dst, const void *src, int elem_bytes, const uint64_t *d_pieces, uint64_t npieces,
                           hrs_stream_t stream);

/* ---- observability ---- */

/* Per-launch device timing for benchmarks (thread-local, off by default).  While
 * enabled, every kernel this thread enqueues is bracketed by CUDA events recorded
 * on the launch stream.  hrs_profile_collect synchronises on those events, writes
 * up to `max` records in launch order, returns how many it wrote, and clears the
 * list.  kind: 0 init, 1 digit histogram (k_hist), 2 rank + look-back + scatter
 * (k_scatter), 3 local sort (pass = size class), 4 copy/fill, 5 bucket
 * classification (k_classify). */
typedef struct {
    int kind;
    int pass;
    float ms;
} hrs_profile_record;
void hrs_profile_enable(int on);
int hrs_profile_collect(hrs_profile_record *out, int max);
/* Number of kernel launches this thread has enqueued through the library. */
uint64_t hrs_launch_count(void);

const char *hrs_status_string(hrs_status status);
int hrs_last_cuda_error(void);
int hrs_version(void);

#if defined(__GNUC__)
#pragma GCC visibility pop
#endif
#ifdef __cplusplus
}
#endif
#endif /* HRS_H_ */
