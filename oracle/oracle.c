/*
 * oracle.c -- plain, slow, obviously-correct CPU oracle for the hybrid radix sort
 * of Stehle & Jacobsen, "A Memory Bandwidth-Efficient Hybrid Radix Sort on GPUs"
 * (arXiv 1611.01137; /root/reference/PAPER.md, cited as P:<line>).
 *
 * TEST INFRASTRUCTURE ONLY.  Only tests/, __graft_entry__.smoke() and bench.py's
 * cpu_baseline / --impl reference legs may load or call this code.  It shares no
 * code, header, table or constant with the CUDA library (paper_1611_01137_b200/),
 * and the library never calls it: there is no CPU fallback.
 *
 * What the method computes: the unique STABLE sort of the
 * records by the key bits [begin, end).  With W = end - begin and
 * sk(x) = (x >> begin) & (2^W - 1), the output is keys_in[pi(i)], vals_in[pi(i)]
 * for the unique permutation pi with (sk(keys_in[pi(i)]), pi(i)) strictly
 * increasing.  The MSD recursion "ultimately yields the sorted sequence"
 * (P:302-303); stability (BJ north_star) makes it unique.
 *
 * Every function works on uint64_t keys and values (callers widen u32 data); all
 * arithmetic is integer, there is no rounding anywhere.
 *
 * Functions and the passages they follow:
 *   oracle_digit_histogram  -- step (1) of a counting sort: the histogram of a
 *                              digit.
 *   oracle_partition_pass   -- one counting sort of the whole input on one digit:
 *                              histogram, exclusive prefix sum -> bucket offsets,
 *                              scatter in input order,
 *                              i.e. one stable pass.
 *   oracle_lsd_sort         -- the LSD radix sort: stable counting passes from the
 *                              least- to the most-significant digit,
 *                              8-bit digits (d = 8), the last one
 *                              narrower when 8 does not divide W.
 *
 * Error behaviour: returns 0 on success, 1 on invalid arguments, 2 when malloc
 * fails.  Nothing is written on error.
 */
#include <stdint.h>
#include <stdlib.h>
#include <string.h>

static uint64_t digit_of(uint64_t key, int lo, int width)
{
    /* bits [lo, lo + width) of key; width in 1..8 so the shift below never hits 64 */
    return (key >> lo) & ((((uint64_t)1) << width) - 1);
}

int oracle_digit_histogram(const uint64_t *keys, uint64_t n, int lo, int hi,
                           uint64_t *hist /* 2^(hi-lo) entries */)
{
    if (lo < 0 || hi > 64 || hi - lo < 1 || hi - lo > 8) return 1;
    int width = hi - lo;
    uint64_t radix = ((uint64_t)1) << width;
    for (uint64_t d = 0; d < radix; d++) hist[d] = 0;
    for (uint64_t i = 0; i < n; i++) hist[digit_of(keys[i], lo, width)]++;
    return 0;
}

int oracle_partition_pass(const uint64_t *keys, const uint64_t *vals, uint64_t n,
                          int lo, int hi, uint64_t *keys_out, uint64_t *vals_out,
                          uint64_t *offsets /* 2^(hi-lo) + 1 entries: bucket starts, then n */)
{
    if (lo < 0 || hi > 64 || hi - lo < 1 || hi - lo > 8) return 1;
    int width = hi - lo;
    uint64_t radix = ((uint64_t)1) << width;
    uint64_t *cnt = (uint64_t *)malloc(sizeof(uint64_t) * radix);
    uint64_t *pos = (uint64_t *)malloc(sizeof(uint64_t) * radix);
    if (!cnt || !pos) { free(cnt); free(pos); return 2; }

    /* (1) histogram */
    for (uint64_t d = 0; d < radix; d++) cnt[d] = 0;
    for (uint64_t i = 0; i < n; i++) cnt[digit_of(keys[i], lo, width)]++;
    /* (2) exclusive prefix sum -> offset of every bucket */
    uint64_t run = 0;
    for (uint64_t d = 0; d < radix; d++) { pos[d] = run; offsets[d] = run; run += cnt[d]; }
    offsets[radix] = run;
    /* (3) scatter, visiting the input in order: equal digits keep input order */
    for (uint64_t i = 0; i < n; i++) {
        uint64_t d = digit_of(keys[i], lo, width);
        keys_out[pos[d]] = keys[i];
        if (vals) vals_out[pos[d]] = vals[i];
        pos[d]++;
    }
    free(cnt);
    free(pos);
    return 0;
}

int oracle_lsd_sort(const uint64_t *keys, const uint64_t *vals, uint64_t n,
                    int begin, int end, uint64_t *keys_out, uint64_t *vals_out)
{
    if (begin < 0 || end > 64 || begin > end) return 1;
    uint64_t *k2 = NULL, *v2 = NULL;
    uint64_t offs[257];
    if (n) {
        k2 = (uint64_t *)malloc(sizeof(uint64_t) * n);
        if (vals) v2 = (uint64_t *)malloc(sizeof(uint64_t) * n);
        if (!k2 || (vals && !v2)) { free(k2); free(v2); return 2; }
    }
    /* the result starts as a copy of the input (identity when begin == end) */
    memcpy(keys_out, keys, sizeof(uint64_t) * n);
    if (vals) memcpy(vals_out, vals, sizeof(uint64_t) * n);

    for (int lo = begin; lo < end; lo += 8) {
        int hi = lo + 8 < end ? lo + 8 : end;
        int rc = oracle_partition_pass(keys_out, vals ? vals_out : NULL, n, lo, hi,
                                       k2 ? k2 : keys_out, v2, offs);
        if (rc) { free(k2); free(v2); return rc; }
        if (n) {
            memcpy(keys_out, k2, sizeof(uint64_t) * n);
            if (vals) memcpy(vals_out, v2, sizeof(uint64_t) * n);
        }
    }
    free(k2);
    free(v2);
    return 0;
}
