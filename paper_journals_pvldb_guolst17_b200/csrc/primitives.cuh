// primitives.cuh -- hand-written device primitives for the batch pipeline:
// LSD radix sort of (u64 key, u32 value) pairs and an exclusive scan of u32
// counts into u64 offsets.  Both are plain multi-CTA kernels (no CUB).
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

namespace ppr {

constexpr int RS_THREADS = 256;
// keys per thread per pass: small batches use short tiles so that many CTAs
// share a pass, large ones long tiles so that the per-tile histograms stay few
inline int rs_items(uint64_t n) { return n <= (1u << 18) ? 2 : 16; }
constexpr uint32_t RS_FUSED_MAX_TILES = 64;  // at most this many tiles: no separate scan kernel
inline uint64_t rs_tiles(uint64_t n) {
    const uint64_t tile = (uint64_t)RS_THREADS * rs_items(n);
    return (n + tile - 1) / tile;
}
// scratch entries (u32) the sort needs for n keys
// (valid for every sort of m <= n keys)
inline uint64_t rs_hist_entries(uint64_t n) {
    uint64_t t = rs_tiles(n), ts = rs_tiles(n < (1u << 18) ? n : (1u << 18));
    const uint64_t one = 256 * ((t > ts ? t : ts) + 1) + 256;
    // chained small sorts (<= RS_FUSED_MAX_TILES tiles) rotate three histograms
    const uint64_t tc = t < RS_FUSED_MAX_TILES ? t : RS_FUSED_MAX_TILES;
    const uint64_t three = 3 * 256 * (tc + 1);
    return one > three ? one : three;
}

// Sorts n pairs by the bits [shift, shift+8) for every shift in `shifts`
// (stable LSD).  Data ping-pongs between (k0,v0) and (k1,v1); returns 0 if
// the result ends in (k0,v0), 1 if in (k1,v1).  `launches` is incremented
// by the number of kernels launched.
int radix_sort_pairs(uint64_t* k0, uint32_t* v0, uint64_t* k1, uint32_t* v1, uint64_t n,
                     const int* shifts, int npasses, uint32_t* hist, cudaStream_t st,
                     uint32_t* launches);

constexpr int SCAN_THREADS = 1024;
constexpr int SCAN_ITEMS = 4;
constexpr int SCAN_TILE = SCAN_THREADS * SCAN_ITEMS;
inline uint64_t scan_parts(uint64_t n) { return (n + SCAN_TILE - 1) / SCAN_TILE; }

// out[i] = sum_{j<i} in[j] (u64), *total = sum of all (device pointer).
// part: scratch of scan_parts(n) + 1 u64.
void exclusive_scan_u32(const uint32_t* in, unsigned long long* out, uint64_t n,
                        unsigned long long* part, unsigned long long* total, cudaStream_t st,
                        uint32_t* launches);

// digit shifts for keys (hi << 32 | lo) with hi, lo < 2^bits
int key_shifts(int bits, int* shifts /* >= 8 */);

// Resident CTAs per SM of kernel `fn` at `threads` threads on the calling
// thread's current device, capped at `cap`: cached per (device, kernel),
// thread-safe (persistent and cooperative grids are sized from it).
cudaError_t blocks_per_sm(const void* fn, int threads, int cap, int* out);

}  // namespace ppr
