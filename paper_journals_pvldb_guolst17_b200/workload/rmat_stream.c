/*
 * rmat_stream.c -- seeded synthetic edge-stream generator (INPUT ONLY).
 *
 * This is the one module both the CUDA product path (via bench.py / tests)
 * and the CPU oracle consume.  It contains none of the PPR method's
 * arithmetic: it only draws arcs.  Recipe:
 *
 *   1. R-MAT [Chakrabarti et al.] at scale = ceil(log2 n): attempt i draws,
 *      for each level l, a uniform from a counter-based hash h(seed, i, l)
 *      and picks a quadrant with probabilities (a, b, c, d).
 *   2. Endpoints >= n are rejected, self-loops dropped, duplicates removed
 *      (directed: key (u,v); undirected: key (min,max)).  Attempts continue
 *      in deterministic chunks until at least m unique arcs exist.
 *   3. Sorting the unique set by a seeded hash tag gives the stream
 *      order ("randomly setting the timestamps"); the
 *      first m are kept.
 *   4. A seeded random relabelling of [0, n) so hub ids are not clustered.
 *
 * Everything is a pure function of (n, m, seed, a, b, c, undirected); the
 * thread count does not change the output.
 */
#include <stdint.h>
#include <stdlib.h>
#include <string.h>
#ifdef _OPENMP
#include <omp.h>
#endif

static inline uint64_t mix64(uint64_t x) { /* splitmix64 finaliser */
    x ^= x >> 30;
    x *= 0xBF58476D1CE4E5B9ULL;
    x ^= x >> 27;
    x *= 0x94D049BB133111EBULL;
    x ^= x >> 31;
    return x;
}

/* counter-based hash of (i, j) under a pre-mixed seed sm = seed_mix(seed) */
static inline uint64_t seed_mix(uint64_t seed) {
    return mix64(seed * 0x9E3779B97F4A7C15ULL + 0x632BE59BD9B4E019ULL);
}
static inline uint64_t hash3(uint64_t sm, uint64_t i, uint64_t j) {
    return mix64(sm ^ (i * 0xD1B54A32D192ED03ULL + j * 0x8CB92BA72F3D8DD7ULL + 1));
}

/* uniform integer in [0, bound) from a hash (multiply-shift; bias < 2^-32) */
static inline uint64_t bounded(uint64_t h, uint64_t bound) {
    return (uint64_t)(((unsigned __int128)h * bound) >> 64);
}

/* ---------------- parallel LSD radix sort (keys, optional u64 payload) ---------------- */
static int radix_sort_u64(uint64_t *keys, uint64_t *vals, uint64_t n, int lo_bit, int hi_bit) {
    if (n < 2) return 0;
    uint64_t *tk = (uint64_t *)malloc(n * sizeof(uint64_t));
    uint64_t *tv = vals ? (uint64_t *)malloc(n * sizeof(uint64_t)) : NULL;
    if (!tk || (vals && !tv)) {
        free(tk);
        free(tv);
        return -1;
    }
    const int DB = 16, NB = 1 << DB;
    int nthreads = 1;
#ifdef _OPENMP
    nthreads = omp_get_max_threads();
#endif
    uint64_t *hist = (uint64_t *)malloc((size_t)nthreads * NB * sizeof(uint64_t));
    if (!hist) {
        free(tk);
        free(tv);
        return -1;
    }
    uint64_t *sk = keys, *dk = tk, *sv = vals, *dv = tv;
    for (int shift = lo_bit; shift < hi_bit; shift += DB) {
        memset(hist, 0, (size_t)nthreads * NB * sizeof(uint64_t));
#pragma omp parallel num_threads(nthreads)
        {
            int t = 0;
#ifdef _OPENMP
            t = omp_get_thread_num();
#endif
            uint64_t lo = n * t / nthreads, hi = n * (t + 1) / nthreads;
            uint64_t *h = hist + (size_t)t * NB;
            for (uint64_t i = lo; i < hi; i++) h[(sk[i] >> shift) & (NB - 1)]++;
#pragma omp barrier
#pragma omp single
            {
                uint64_t run = 0;
                for (int d = 0; d < NB; d++)
                    for (int tt = 0; tt < nthreads; tt++) {
                        uint64_t c = hist[(size_t)tt * NB + d];
                        hist[(size_t)tt * NB + d] = run;
                        run += c;
                    }
            }
            for (uint64_t i = lo; i < hi; i++) {
                uint64_t k = sk[i];
                uint64_t p = h[(k >> shift) & (NB - 1)]++;
                dk[p] = k;
                if (sv) dv[p] = sv[i];
            }
        }
        uint64_t *sw = sk;
        sk = dk;
        dk = sw;
        sw = sv;
        sv = dv;
        dv = sw;
    }
    if (sk != keys) {
        memcpy(keys, sk, n * sizeof(uint64_t));
        if (vals) memcpy(vals, sv, n * sizeof(uint64_t));
    }
    free(hist);
    free(tk);
    free(tv);
    return 0;
}

static uint64_t unique_sorted(uint64_t *k, uint64_t n) {
    if (n == 0) return 0;
    uint64_t w = 1;
    for (uint64_t i = 1; i < n; i++)
        if (k[i] != k[w - 1]) k[w++] = k[i];
    return w;
}

/* Draw attempts [first, first+count) into out[0..count); rejected attempts
 * become `sentinel`, a key larger than every valid key. */
static void draw(uint64_t sm, uint64_t first, uint64_t count, uint32_t n, int scale,
                 double a, double b, double c, int undirected, uint64_t sentinel,
                 uint64_t *out) {
    const uint64_t ta = (uint64_t)(a * 4294967296.0);
    const uint64_t tb = (uint64_t)((a + b) * 4294967296.0);
    const uint64_t tc = (uint64_t)((a + b + c) * 4294967296.0);
#pragma omp parallel for schedule(static)
    for (int64_t ii = 0; ii < (int64_t)count; ii++) {
        uint64_t i = first + (uint64_t)ii;
        uint64_t u = 0, v = 0, h = 0;
        for (int l = 0; l < scale; l++) {
            if ((l & 1) == 0) h = hash3(sm, i, (uint64_t)(l >> 1));
            uint64_t r = (l & 1) ? (h >> 32) : (h & 0xFFFFFFFFULL);
            int ub, vb;
            if (r < ta) { ub = 0; vb = 0; }
            else if (r < tb) { ub = 0; vb = 1; }
            else if (r < tc) { ub = 1; vb = 0; }
            else { ub = 1; vb = 1; }
            u = (u << 1) | (uint64_t)ub;
            v = (v << 1) | (uint64_t)vb;
        }
        int good = (u < n) && (v < n) && (u != v);
        if (undirected && u > v) {
            uint64_t t = u;
            u = v;
            v = t;
        }
        out[ii] = good ? ((u << 32) | v) : sentinel;
    }
}

/*
 * Fills src[m], dst[m] (stream order).  For undirected streams each entry is
 * one undirected edge {src, dst}.  Returns 0, or -1 on bad arguments /
 * allocation failure, or -2 if m unique arcs could not be found.
 */
int rmat_stream(uint32_t n, uint64_t m, uint64_t seed, double a, double b, double c,
                int undirected, uint32_t *src, uint32_t *dst) {
    if (n < 2 || a < 0 || b < 0 || c < 0 || a + b + c > 1.0) return -1;
    int scale = 0;
    while ((1ULL << scale) < n) scale++;
    uint64_t maxpairs = undirected ? (uint64_t)n * (n - 1) / 2 : (uint64_t)n * (n - 1);
    if (m > maxpairs) return -1;
    const uint64_t sm = seed_mix(seed);
    const int key_bits = 32 + scale;
    const uint64_t sentinel = (((1ULL << scale) - 1) << 32) | 0xFFFFFFFFULL;
    uint64_t nk = 0, drawn = 0, chunk = m + m / 3 + 1024;
    uint64_t *keys = NULL;
    for (int round = 0; round < 64; round++) {
        uint64_t *nkp = (uint64_t *)realloc(keys, (nk + chunk) * sizeof(uint64_t));
        if (!nkp) {
            free(keys);
            return -1;
        }
        keys = nkp;
        draw(sm, drawn, chunk, n, scale, a, b, c, undirected, sentinel, keys + nk);
        drawn += chunk;
        nk += chunk;
        if (radix_sort_u64(keys, NULL, nk, 0, key_bits) != 0) {
            free(keys);
            return -1;
        }
        nk = unique_sorted(keys, nk);
        if (nk && keys[nk - 1] == sentinel) nk--;
        if (nk >= m) break;
        chunk = (m - nk) + (m - nk) / 2 + 1024;
    }
    if (nk < m) {
        free(keys);
        return -2;
    }
    /* stream order: sort the unique set by a seeded 48-bit hash tag (a random
     * permutation; tag ties keep key order, so the result is deterministic) */
    uint64_t sseed = seed_mix(seed ^ 0x5EED0F5EED0F5EEDULL);
    uint64_t *tags = (uint64_t *)malloc(nk * sizeof(uint64_t));
    if (!tags) {
        free(keys);
        return -1;
    }
#pragma omp parallel for schedule(static)
    for (int64_t i = 0; i < (int64_t)nk; i++) tags[i] = hash3(sseed, keys[i], 7) >> 16;
    if (radix_sort_u64(tags, keys, nk, 0, 48) != 0) {
        free(tags);
        free(keys);
        return -1;
    }
    free(tags);
    /* relabelling permutation of [0, n) */
    uint32_t *perm = (uint32_t *)malloc((size_t)n * sizeof(uint32_t));
    if (!perm) {
        free(keys);
        return -1;
    }
    for (uint32_t i = 0; i < n; i++) perm[i] = i;
    uint64_t pseed = seed_mix(seed ^ 0x0BADC0DE0BADC0DEULL);
    for (uint32_t i = n - 1; i > 0; i--) {
        uint32_t j = (uint32_t)bounded(hash3(pseed, i, 11), (uint64_t)i + 1);
        uint32_t t = perm[i];
        perm[i] = perm[j];
        perm[j] = t;
    }
#pragma omp parallel for schedule(static)
    for (int64_t i = 0; i < (int64_t)m; i++) {
        src[i] = perm[(uint32_t)(keys[i] >> 32)];
        dst[i] = perm[(uint32_t)(keys[i] & 0xFFFFFFFFULL)];
    }
    free(perm);
    free(keys);
    return 0;
}
