// decode.cuh — device-side CGR codeword decoding for sm_100a (FORMAT.md R1-R19): the 64-bit window decoder and the
// warp-parallel decoder of Alg. 4 (test hook; the production path reads records through BitReader, device.cuh).
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
// Fast path in 32-bit arithmetic: the top 32 bits of the window (one funnel shift of the two words holding it) hold
// every codeword of at most 32 bits (zeta_3: values < 2^24; gamma: < 2^15), i.e. nearly all gaps and counts; longer
// codewords take the 64-bit window, then the bit-serial slow path.
template <int K>
__device__ __forceinline__ uint64_t decode(const uint64_t* __restrict__ W, uint64_t& p) {
    const uint64_t i = p >> 6;
    const uint32_t s = (uint32_t)(p & 63);
    const uint64_t a = ldg64(W + i), b = ldg64(W + i + 1);
    const uint32_t x = s < 32 ? (uint32_t)(a >> 32) : (uint32_t)a;
    const uint32_t y = s < 32 ? (uint32_t)a : (uint32_t)(b >> 32);
    const uint32_t hi = __funnelshift_l(y, x, s & 31);  // window bits 0..31
    const uint32_t z = __clz(hi);
    if (K == 1) {
        if (z < 16) {
            const uint32_t L = 2 * z + 1;
            p += L;
            return hi >> (32 - L);
        }
    } else {
        const uint32_t h = z + 1, L = h * (K + 1);
        if (L <= 32) {
            p += L;
            return (hi << h) >> (32 - K * h);
        }
    }
    const uint64_t win = s ? (a << s) | (b >> (64 - s)) : a;
    const uint32_t zz = (uint32_t)__clzll((long long)win);
    if (K == 1) {
        if (zz < 32) {
            const uint32_t L = 2 * zz + 1;
            p += L;
            return win >> (64 - L);
        }
    } else {
        const uint32_t h = zz + 1, L = h * (K + 1);
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

}  // namespace gcgt_dev

namespace gcgt_dev {

// Speculative decode for the warp-parallel decoder: the codeword's length, or 0xFFFF when it does not fit the
// 64-bit window path (then only the exact slow path can decode it).
template <int K>
__device__ __forceinline__ uint32_t spec_decode(const uint64_t* __restrict__ W, uint64_t q, uint64_t& val) {
    const uint64_t win = window(W, q);
    const uint32_t z = (uint32_t)__clzll((long long)win);
    if (K == 1) {
        if (z < 32) {
            const uint32_t L = 2 * z + 1;
            val = win >> (64 - L);
            return L;
        }
    } else {
        const uint32_t h = z + 1, L = h * (K + 1);
        if (L <= 64) {
            val = (win << h) >> (64 - K * h);
            return L;
        }
    }
    val = 0;
    return 0xFFFFu;
}

// One window step of Alg. 4 parallelDecode, B200 form, over WIN <= 32 lanes: lane i decodes
// speculatively at p+i (lines 5-7); the valid starts are marked from lane 0 by pointer jumping (lines 9-15,
// Fig. 5): each marked lane marks the start its pointer names (__reduce_or_sync of one-hot masks), then every
// pointer jumps to its target's pointer; 'x' (>= WIN) propagates.  By Lemma 5.2 five rounds cover 32 lanes.
// Returns the mask of lanes holding a valid codeword start; val/len are the lane's speculative decode.
// With TRACE, trace_pos/trace_flags receive the per-round state (row 0 = initial) and *rounds the row count.
template <int K, int WIN, bool TRACE>
__device__ __forceinline__ uint32_t window_step(const uint64_t* __restrict__ W, uint64_t p, uint64_t& val,
                                                uint32_t& len, uint32_t* trace_pos = nullptr,
                                                uint32_t* trace_flags = nullptr, uint32_t* rounds = nullptr) {
    const uint32_t lane = threadIdx.x & 31;
    len = spec_decode<K>(W, p + lane, val);
    uint32_t pos = lane < (uint32_t)WIN ? lane + len : 0xFFFFFFFFu;  // start of the following codeword
    uint32_t flags = 1u;                                             // lane 0 starts a codeword (line 8)
    if (TRACE && lane < (uint32_t)WIN) { trace_pos[lane] = pos; trace_flags[lane] = lane == 0; }
    int r = 0;
#pragma unroll
    for (; r < 5; r++) {
        const uint32_t mark = (((flags >> lane) & 1u) && pos < (uint32_t)WIN) ? (1u << pos) : 0u;
        const uint32_t m = __reduce_or_sync(0xffffffffu, mark);
        if (!m) break;  // line 12: no marked lane points inside the window
        flags |= m;
        const uint32_t pp = __shfl_sync(0xffffffffu, pos, pos & 31);
        pos = pos < (uint32_t)WIN ? pp : 0xFFFFFFFFu;
        if (TRACE && lane < (uint32_t)WIN) {
            trace_pos[(r + 1) * 32 + lane] = pos;
            trace_flags[(r + 1) * 32 + lane] = (flags >> lane) & 1u;
        }
    }
    if (TRACE && lane == 0) *rounds = (uint32_t)r + 1;
    return flags;
}

// Decodes `count` consecutive codewords from bit p with the whole warp (window_step per 32 bits).  The first
// min(#valid, remaining) codewords of each step are handed to fn(step_base, take, index, value, active)
// warp-uniformly (lines 16-17).  Returns the bit after the last codeword.  All 32 lanes must call it with
// warp-uniform p and count.
template <int K, class Fn>
__device__ __forceinline__ uint64_t warp_decode(const uint64_t* __restrict__ W, uint64_t p, uint64_t count, Fn&& fn) {
    const uint32_t lane = threadIdx.x & 31;
    uint32_t lt;
    asm("mov.u32 %0, %%lanemask_lt;" : "=r"(lt));
    uint64_t done = 0;
    while (done < count) {
        uint64_t val;
        uint32_t len;
        const uint32_t flags = window_step<K, 32, false>(W, p, val, len);
        const uint64_t rem = count - done;
        const uint32_t nvalid = __popc(flags);
        const uint32_t take = (uint64_t)nvalid < rem ? nvalid : (uint32_t)rem;
        const uint32_t last = (uint32_t)__fns(flags, 0, (int)take);
        uint32_t last_len = __shfl_sync(0xffffffffu, len, last);
        if (last_len == 0xFFFFu) {  // only the last valid codeword can be this long: decode it exactly
            uint64_t q = p + last;
            const uint64_t v = decode_slow<K>(W, q);
            if (lane == last) val = v;
            last_len = (uint32_t)(q - (p + last));
        }
        const uint32_t idx = __popc(flags & lt);
        const bool act = ((flags >> lane) & 1u) && idx < take;
        fn(done, take, done + idx, val, act);
        p += last + last_len;
        done += take;
    }
    return p;
}

}  // namespace gcgt_dev
