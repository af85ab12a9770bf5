// internal.h — product-internal declarations shared by encode.cpp and gcgt.cu (NOT part of the C ABI;
// the oracle never includes this).
#pragma once
#include <stdint.h>

#include <string>
#include <vector>

#include "../../include/gcgt.h"

// Host CGR object.  `words` holds the canonical byte stream (FORMAT.md R1) in memory order, padded with at least
// two zero 64-bit words so that device 128-bit window loads never run off the end.
struct gcgt_cgr {
    uint64_t n = 0;        // records held (vertices base .. base + n - 1)
    uint64_t base = 0;     // first vertex (0 for a whole graph; a vertex-range slice otherwise)
    uint64_t n_total = 0;  // vertices of the whole graph (ids < n_total); == n for a whole graph
    uint64_t nbits = 0;
    gcgt_params params{};
    std::vector<uint64_t> words;        // ceil(nbits/64) + 2 words; bytes = (uint8_t*)words.data()
    std::vector<uint64_t> bit_offsets;  // n + 1
    uint64_t nbytes() const { return (nbits + 7) / 8; }
};

namespace gcgt_internal {
gcgt_status fail(gcgt_status st, const std::string& msg);  // records the thread-local message, returns st
void clear_error();
}  // namespace gcgt_internal
