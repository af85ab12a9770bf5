// internal.h — product-internal declarations shared by encode.cpp and gcgt.cu (NOT part of the C ABI;
// the oracle never includes this).
#pragma once
#include <stdint.h>

#include <memory>
#include <mutex>
#include <string>
#include <utility>
#include <vector>

#include "../../include/gcgt.h"

// Derived load tables of a whole CGR (gcgt.cu builds them on the first gcgt_load of the whole CGR, or on
// gcgt_cgr_pin, and keeps them with the CGR so that later loads are plain host-to-device copies): the compact bit
// offsets and the interval checkpoint table.  Device-independent host arrays; `pinned` lists the ranges
// gcgt_cgr_pin page-locked (released by gcgt_cgr_free).
struct gcgt_cgr_tables {
    bool compact = false;          // compact offsets fit (every 256-vertex block spans < 2^32 bits)
    std::vector<uint64_t> anc;     // u64 anchor per 256 vertices
    std::vector<uint32_t> rel;     // u32 per vertex (n + 1), relative to its anchor
    bool ck_built = false;
    uint32_t ck_c = 0;             // intervals per chunk the checkpoint table was built for
    uint64_t rows = 0, chunks = 0;
    std::vector<uint32_t> wptr, bits, ck0, ilen, prev;
    std::vector<uint64_t> after, pos;
    std::vector<std::pair<void*, size_t>> pinned;
};

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
    mutable std::mutex mu;                          // guards `tables`
    mutable std::unique_ptr<gcgt_cgr_tables> tables;  // built lazily (gcgt.cu)
};

namespace gcgt_internal {
gcgt_status fail(gcgt_status st, const std::string& msg);  // records the thread-local message, returns st
void clear_error();
void release_tables(gcgt_cgr* c);  // gcgt.cu: unpins and frees the derived tables (gcgt_cgr_free)
}  // namespace gcgt_internal
