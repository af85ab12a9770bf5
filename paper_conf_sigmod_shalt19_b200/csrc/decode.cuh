// decode.cuh — device-side CGR decoding for sm_100a (FORMAT.md R1-R19).
//
// The device keeps the CGR as 64-bit words in stream order (bit i of the stream is bit 63-(i%64) of word i/64;
// the load step byte-swaps the canonical MSB-first bytes once).  A codeword at bit p is decoded from a 64-bit
// window W[p/64] << (p%64) | W[p/64+1] >> (64 - p%64): one CLZ gives the unary part (App. B),
// one shift pair gives the payload.  gamma codes longer than 63 bits and zeta codes longer than 64 bits take a
// (never-taken on our workloads) slow path.
#pragma once
#include <stdint.h>

namespace gcgt_dev {

__device__ __forceinline__ uint64_t ldg64(const uint64_t* p) { return __ldg(reinterpret_cast<const unsigned long long*>(p)); }

__device__ __forceinline__ uint64_t window(const uint64_t* __restrict__ W, uint64_t p) {
    const uint64_t i = p >> 6;
    const uint32_t s = (uint32_t)(p & 63);
    const uint64_t a = ldg64(W + i), b = ldg64(W + i + 1);
    return s ? (a << s) | (b >> (64 - s)) : a;
}

__device__ __forceinline__ int stream_bit(const uint64_t* __restrict__ W, uint64_t p) {
    return (int)((ldg64(W + (p >> 6)) >> (63 - (p & 63))) & 1);
}

// Slow path: codes whose length exceeds the 64-bit window (gamma >= 64 bits: x >= 2^32; zeta: x >= 2^48).
template <int K>
__device__ __noinline__ uint64_t decode_slow(const uint64_t* __restrict__ W, uint64_t& p) {
    uint64_t z = 0;
    while (!stream_bit(W, p)) { z++; p++; }
    uint64_t payload;
    if (K == 1) payload = z + 1;
    else { p++; payload = (z + 1) * K; }
    uint64_t x = 0;
    for (uint64_t i = 0; i < payload; i++) x = (x << 1) | (uint64_t)stream_bit(W, p + i);
    p += payload;
    return x;
}

// decodeNum (Alg. 1 l.6): one VLC codeword at p; advances p.
template <int K>
__device__ __forceinline__ uint64_t decode(const uint64_t* __restrict__ W, uint64_t& p) {
    const uint64_t win = window(W, p);
    const uint32_t z = (uint32_t)__clzll((long long)win);
    if (K == 1) {
        if (z < 32) {
            const uint32_t L = 2 * z + 1;
            p += L;
            return win >> (64 - L);
        }
    } else {
        const uint32_t h = z + 1, L = h * (K + 1);
        if (L <= 64) {
            p += L;
            return (win << h) >> (64 - K * h);
        }
    }
    return decode_slow<K>(W, p);
}

// Inverse of the first-gap sign map + 1 (App. C :2101-2106, FORMAT.md R9/R11/R17): code c -> u + delta.
__device__ __forceinline__ int64_t unmap_first(uint64_t u, uint64_t c) {
    const uint64_t z = c - 1;
    return (int64_t)u + ((z & 1) ? -(int64_t)(z >> 1) : (int64_t)(z >> 1));
}

// Walks u's record: calls vis.range(start, len) per interval and vis.one(v) per residual.
// Unsegmented (SEG=false): R8-R12.  Segmented (SEG=true): R14-R17.  Returns the neighbour count.
template <int K, bool SEG, class Visitor>
__device__ __forceinline__ uint32_t walk_record(const uint64_t* __restrict__ W, uint64_t p, uint64_t u,
                                                uint32_t min_len, uint32_t seg_bits, Visitor& vis) {
    uint64_t deg = 0;
    if (!SEG) deg = decode<K>(W, p) - 1;
    const uint64_t itv = decode<K>(W, p) - 1;
    uint64_t got = 0;
    int64_t prev_end = 0;
    for (uint64_t t = 0; t < itv; t++) {
        const uint64_t g = decode<K>(W, p);
        const uint64_t len = decode<K>(W, p) - 1 + min_len;
        const int64_t start = t == 0 ? unmap_first(u, g) : prev_end + (int64_t)g;
        vis.range((uint32_t)start, (uint32_t)len);
        prev_end = start + (int64_t)len - 1;
        got += len;
    }
    if (!SEG) {
        const uint64_t nres = deg - got;
        int64_t cur = 0;
        for (uint64_t t = 0; t < nres; t++) {
            const uint64_t c = decode<K>(W, p);
            cur = t == 0 ? unmap_first(u, c) : cur + (int64_t)c;
            vis.one((uint32_t)cur);
        }
        return (uint32_t)deg;
    } else {
        const uint64_t nseg = decode<K>(W, p) - 1;
        const uint64_t base = p;
        for (uint64_t s = 0; s < nseg; s++) {
            uint64_t q = base + s * seg_bits;
            const uint64_t cnt = decode<K>(W, q) - 1;
            int64_t cur = unmap_first(u, decode<K>(W, q));
            vis.one((uint32_t)cur);
            for (uint64_t t = 1; t < cnt; t++) {
                cur += (int64_t)decode<K>(W, q);
                vis.one((uint32_t)cur);
            }
            got += cnt;
        }
        return (uint32_t)got;
    }
}

}  // namespace gcgt_dev
