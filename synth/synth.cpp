// synth.cpp — seeded synthetic graph generators (inputs only; no CGR / BFS / CC / BC arithmetic).
//
// Shared by the oracle side and the product side as INPUT: every graph is a plain CSR (u64 row offsets, u32
// strictly increasing columns).  Recipes follow SURVEY.md §8(d) / DESIGN.md §4, shaped like the paper's
// workloads (Table 1):
//   syn_rmat    R-MAT / Kronecker, Graph500 probabilities, symmetrised, self-loops dropped (configs 1 and 5)
//   syn_web     host-clustered "web" digraph (uk-2002 / uk-2007 shape), BFS-order relabelled (:2275-2276)
//   syn_social  power-law "social" digraph with heavy out-degree skew (twitter-2010 shape), BFS-order relabelled
// Randomness is counter-based (SplitMix64 of (seed, stream, counter)), so the output is independent of the
// OpenMP thread count.
#include <omp.h>
#include <stdint.h>
#include <stdlib.h>
#include <string.h>

#include <algorithm>
#include <atomic>
#include <cmath>
#include <new>
#include <vector>

namespace {

inline uint64_t splitmix(uint64_t x) {
    x += 0x9E3779B97F4A7C15ull;
    x = (x ^ (x >> 30)) * 0xBF58476D1CE4E5B9ull;
    x = (x ^ (x >> 27)) * 0x94D049BB133111EBull;
    return x ^ (x >> 31);
}

struct Rng {  // one stream per (seed, stream id); deterministic sequence
    uint64_t s;
    Rng(uint64_t seed, uint64_t stream) : s(splitmix(seed * 0x632BE59BD9B4E019ull ^ splitmix(stream + 0x1234567ull))) {}
    uint64_t next() { s += 0x9E3779B97F4A7C15ull; return splitmix(s); }
    double unif() { return (double)(next() >> 11) * (1.0 / 9007199254740992.0); }  // [0,1)
    uint64_t below(uint64_t n) { return n ? (uint64_t)(unif() * (double)n) % n : 0; }
};

struct Graph {
    uint64_t n = 0;
    std::vector<uint64_t> rowoff;
    std::vector<uint32_t> cols;
};

// Sort + dedupe each row in place, then compact into a CSR.  rows[u] holds unsorted targets.
void rows_to_csr(uint64_t n, std::vector<std::vector<uint32_t>>& rows, Graph& g, bool drop_self) {
    g.n = n;
    g.rowoff.assign(n + 1, 0);
#pragma omp parallel for schedule(dynamic, 1024)
    for (int64_t u = 0; u < (int64_t)n; u++) {
        auto& r = rows[u];
        if (drop_self) r.erase(std::remove(r.begin(), r.end(), (uint32_t)u), r.end());
        std::sort(r.begin(), r.end());
        r.erase(std::unique(r.begin(), r.end()), r.end());
        g.rowoff[u + 1] = r.size();
    }
    for (uint64_t u = 0; u < n; u++) g.rowoff[u + 1] += g.rowoff[u];
    g.cols.resize(g.rowoff[n]);
#pragma omp parallel for schedule(dynamic, 1024)
    for (int64_t u = 0; u < (int64_t)n; u++) {
        std::copy(rows[u].begin(), rows[u].end(), g.cols.begin() + g.rowoff[u]);
        std::vector<uint32_t>().swap(rows[u]);
    }
}

// BFS-order relabelling (BFSOrder): visit from vertex 0 over out-arcs, restart from the
// smallest unvisited id; new id = visit rank.  Rows are then remapped and re-sorted.
void bfs_relabel(Graph& g) {
    const uint64_t n = g.n;
    std::vector<uint32_t> order;
    order.reserve(n);
    std::vector<uint32_t> newid(n, UINT32_MAX);
    uint64_t next_root = 0;
    while (order.size() < n) {
        while (newid[next_root] != UINT32_MAX) next_root++;
        uint64_t head = order.size();
        newid[next_root] = (uint32_t)order.size();
        order.push_back((uint32_t)next_root);
        while (head < order.size()) {
            uint32_t u = order[head++];
            for (uint64_t e = g.rowoff[u]; e < g.rowoff[u + 1]; e++) {
                uint32_t v = g.cols[e];
                if (newid[v] == UINT32_MAX) { newid[v] = (uint32_t)order.size(); order.push_back(v); }
            }
        }
    }
    std::vector<uint64_t> ro(n + 1, 0);
    for (uint64_t nu = 0; nu < n; nu++) ro[nu + 1] = ro[nu] + (g.rowoff[order[nu] + 1] - g.rowoff[order[nu]]);
    std::vector<uint32_t> co(g.cols.size());
#pragma omp parallel for schedule(dynamic, 4096)
    for (int64_t nu = 0; nu < (int64_t)n; nu++) {
        uint32_t u = order[nu];
        uint64_t o = ro[nu];
        for (uint64_t e = g.rowoff[u]; e < g.rowoff[u + 1]; e++) co[o++] = newid[g.cols[e]];
        std::sort(co.begin() + ro[nu], co.begin() + ro[nu + 1]);
    }
    g.rowoff.swap(ro);
    g.cols.swap(co);
}

// Power-law integer in [lo, hi] with density ~ x^-alpha (inverse-CDF of a continuous Pareto, truncated).
inline double pareto(Rng& r, double lo, double hi, double alpha) {
    double a1 = 1.0 - alpha;
    double u = r.unif();
    if (std::fabs(a1) < 1e-9) return std::exp(std::log(lo) + u * (std::log(hi + 1.0) - std::log(lo)));  // 1/x
    double lo_a = std::pow(lo, a1), hi_a = std::pow(hi + 1.0, a1);
    return std::pow(lo_a + u * (hi_a - lo_a), 1.0 / a1);
}

}  // namespace

extern "C" {

typedef struct syn_graph syn_graph;

uint64_t syn_n(const syn_graph* h) { return ((const Graph*)h)->n; }
uint64_t syn_m(const syn_graph* h) { return ((const Graph*)h)->rowoff.back(); }
void syn_copy(const syn_graph* h, uint64_t* rowoff, uint32_t* cols) {
    const Graph* g = (const Graph*)h;
    memcpy(rowoff, g->rowoff.data(), sizeof(uint64_t) * (g->n + 1));
    const uint64_t m = g->rowoff.back();
    const int64_t chunk = 1 << 22;
#pragma omp parallel for schedule(static)
    for (int64_t c = 0; c < (int64_t)((m + chunk - 1) / chunk); c++) {
        uint64_t b = (uint64_t)c * chunk, e = std::min<uint64_t>(m, b + chunk);
        memcpy(cols + b, g->cols.data() + b, sizeof(uint32_t) * (e - b));
    }
}
void syn_free(syn_graph* h) { delete (Graph*)h; }
int syn_threads(void) { return omp_get_max_threads(); }

// R-MAT (Chakrabarti et al.; Graph500 A=.57 B=.19 C=.19 D=.05): edgefactor * 2^scale generated edges; self-loops
// dropped; symmetrised; deduplicated; rows sorted.  Edge i uses stream i, so the graph does not depend on threads.
syn_graph* syn_rmat(int scale, int edgefactor, uint64_t seed, double A, double B, double C) {
    try {
        const uint64_t n = 1ull << scale, E = (uint64_t)edgefactor << scale;
        std::vector<uint64_t> cnt(n + 1, 0);
        std::vector<uint32_t> es(E), ed(E);
#pragma omp parallel for schedule(static)
        for (int64_t i = 0; i < (int64_t)E; i++) {
            Rng r(seed, (uint64_t)i);
            uint64_t s = 0, d = 0;
            for (int b = 0; b < scale; b++) {
                double p = r.unif();
                int q = p < A ? 0 : p < A + B ? 1 : p < A + B + C ? 2 : 3;
                s = (s << 1) | (uint64_t)(q >> 1);
                d = (d << 1) | (uint64_t)(q & 1);
            }
            es[i] = (uint32_t)s;
            ed[i] = (uint32_t)d;
        }
        std::vector<std::vector<uint32_t>> rows(n);
        // bucket by source (both directions), then sort/dedupe per row
        std::vector<std::atomic<uint32_t>> deg(n);
        for (auto& x : deg) x.store(0, std::memory_order_relaxed);
#pragma omp parallel for schedule(static)
        for (int64_t i = 0; i < (int64_t)E; i++) {
            if (es[i] == ed[i]) continue;
            deg[es[i]].fetch_add(1, std::memory_order_relaxed);
            deg[ed[i]].fetch_add(1, std::memory_order_relaxed);
        }
        std::vector<uint64_t> off(n + 1, 0);
        for (uint64_t u = 0; u < n; u++) off[u + 1] = off[u] + deg[u].load();
        std::vector<uint32_t> flat(off[n]);
        std::vector<std::atomic<uint64_t>> pos(n);
        for (uint64_t u = 0; u < n; u++) pos[u].store(off[u], std::memory_order_relaxed);
#pragma omp parallel for schedule(static)
        for (int64_t i = 0; i < (int64_t)E; i++) {
            if (es[i] == ed[i]) continue;
            flat[pos[es[i]].fetch_add(1)] = ed[i];
            flat[pos[ed[i]].fetch_add(1)] = es[i];
        }
        std::vector<uint32_t>().swap(es);
        std::vector<uint32_t>().swap(ed);
#pragma omp parallel for schedule(dynamic, 1024)
        for (int64_t u = 0; u < (int64_t)n; u++) rows[u].assign(flat.begin() + off[u], flat.begin() + off[u + 1]);
        std::vector<uint32_t>().swap(flat);
        Graph* g = new Graph();
        rows_to_csr(n, rows, *g, true);
        return (syn_graph*)g;
    } catch (...) {
        return nullptr;
    }
}

// One vertex-range slice [lo, hi) of the same symmetrised R-MAT graph (syn_rmat), without materialising the rest:
// every rank (or every pass of a single host) regenerates all edges from the counter-based streams and keeps the
// arcs whose source lies in its range.  Rows are global ids, sorted and deduplicated, self-loops dropped; the rows of
// consecutive slices concatenate to syn_rmat's CSR exactly (C5 at scale 29: 8.6B edges never held at once).
syn_graph* syn_rmat_slice(int scale, int edgefactor, uint64_t seed, double A, double B, double C, uint64_t lo,
                          uint64_t hi) {
    try {
        const uint64_t n = 1ull << scale, E = (uint64_t)edgefactor << scale;
        if (hi > n) hi = n;
        if (lo > hi) lo = hi;
        const uint64_t nr = hi - lo;
        auto edge = [&](uint64_t i, uint64_t& s, uint64_t& d) {
            Rng r(seed, i);
            s = d = 0;
            for (int b = 0; b < scale; b++) {
                double p = r.unif();
                int q = p < A ? 0 : p < A + B ? 1 : p < A + B + C ? 2 : 3;
                s = (s << 1) | (uint64_t)(q >> 1);
                d = (d << 1) | (uint64_t)(q & 1);
            }
        };
        std::vector<std::atomic<uint64_t>> cnt(nr + 1);
        for (auto& x : cnt) x.store(0, std::memory_order_relaxed);
#pragma omp parallel for schedule(static)
        for (int64_t i = 0; i < (int64_t)E; i++) {
            uint64_t s, d;
            edge((uint64_t)i, s, d);
            if (s == d) continue;
            if (s >= lo && s < hi) cnt[s - lo].fetch_add(1, std::memory_order_relaxed);
            if (d >= lo && d < hi) cnt[d - lo].fetch_add(1, std::memory_order_relaxed);
        }
        std::vector<uint64_t> off(nr + 1, 0);
        for (uint64_t u = 0; u < nr; u++) off[u + 1] = off[u] + cnt[u].load();
        std::vector<uint32_t> flat(off[nr]);
        for (uint64_t u = 0; u < nr; u++) cnt[u].store(off[u], std::memory_order_relaxed);
#pragma omp parallel for schedule(static)
        for (int64_t i = 0; i < (int64_t)E; i++) {
            uint64_t s, d;
            edge((uint64_t)i, s, d);
            if (s == d) continue;
            if (s >= lo && s < hi) flat[cnt[s - lo].fetch_add(1)] = (uint32_t)d;
            if (d >= lo && d < hi) flat[cnt[d - lo].fetch_add(1)] = (uint32_t)s;
        }
        Graph* g = new Graph();
        g->n = nr;
        g->rowoff.assign(nr + 1, 0);
#pragma omp parallel for schedule(dynamic, 1024)
        for (int64_t u = 0; u < (int64_t)nr; u++) {
            uint32_t* b = flat.data() + off[u];
            uint32_t* e = flat.data() + off[u + 1];
            std::sort(b, e);
            g->rowoff[u + 1] = (uint64_t)(std::unique(b, e) - b);
        }
        for (uint64_t u = 0; u < nr; u++) g->rowoff[u + 1] += g->rowoff[u];
        g->cols.resize(g->rowoff[nr]);
#pragma omp parallel for schedule(dynamic, 1024)
        for (int64_t u = 0; u < (int64_t)nr; u++)
            std::copy(flat.begin() + off[u], flat.begin() + off[u] + (g->rowoff[u + 1] - g->rowoff[u]),
                      g->cols.begin() + g->rowoff[u]);
        return (syn_graph*)g;
    } catch (...) {
        return nullptr;
    }
}

// Per-vertex arc counts of the symmetrised R-MAT graph before deduplication (an upper bound on the degree), for
// choosing arc-balanced vertex-range slices without generating the graph.
int syn_rmat_counts(int scale, int edgefactor, uint64_t seed, double A, double B, double C, uint32_t* counts) {
    const uint64_t n = 1ull << scale, E = (uint64_t)edgefactor << scale;
    std::atomic<uint32_t>* c = reinterpret_cast<std::atomic<uint32_t>*>(counts);
#pragma omp parallel for schedule(static)
    for (int64_t v = 0; v < (int64_t)n; v++) counts[v] = 0;
#pragma omp parallel for schedule(static)
    for (int64_t i = 0; i < (int64_t)E; i++) {
        Rng r(seed, (uint64_t)i);
        uint64_t s = 0, d = 0;
        for (int b = 0; b < scale; b++) {
            double p = r.unif();
            int q = p < A ? 0 : p < A + B ? 1 : p < A + B + C ? 2 : 3;
            s = (s << 1) | (uint64_t)(q >> 1);
            d = (d << 1) | (uint64_t)(q & 1);
        }
        if (s == d) continue;
        c[s].fetch_add(1, std::memory_order_relaxed);
        c[d].fetch_add(1, std::memory_order_relaxed);
    }
    return 0;
}

// Host-clustered web digraph (uk-2002 / uk-2007 shape):
//  * hosts = contiguous id ranges, sizes power-law (alpha 1.6) in [4, 1e5];
//  * out-degree power-law (alpha 2.1) in [1, 5000], ~8% dangling pages, rescaled to mean_deg;
//  * arcs: ~70% in runs of consecutive ids inside the host (mean run 12), ~25% uniform inside the host,
//    ~5% to a random page of another host chosen preferentially (Zipf over hosts);
//  * then BFS-order relabelling.
syn_graph* syn_web(uint64_t n, double mean_deg, uint64_t seed, int relabel) {
    try {
        // hosts (sequential; cheap)
        std::vector<uint32_t> host_start;
        {
            Rng r(seed, 0xB0057ull);
            uint64_t p = 0;
            while (p < n) {
                uint64_t sz = (uint64_t)pareto(r, 4.0, 1e5, 1.6);
                host_start.push_back((uint32_t)p);
                p += sz;
            }
            host_start.push_back((uint32_t)n);
        }
        const uint64_t H = host_start.size() - 1;
        // raw degrees, then rescale to mean_deg
        std::vector<double> raw(n);
        double sum = 0.0;
#pragma omp parallel for reduction(+ : sum) schedule(static)
        for (int64_t u = 0; u < (int64_t)n; u++) {
            Rng r(seed, 0x100000000ull + (uint64_t)u);
            raw[u] = r.unif() < 0.08 ? 0.0 : pareto(r, 1.0, 5000.0, 2.1);
            sum += raw[u];
        }
        const double scale = mean_deg * (double)n / sum;
        std::vector<std::vector<uint32_t>> rows(n);
#pragma omp parallel for schedule(dynamic, 256)
        for (int64_t uu = 0; uu < (int64_t)n; uu++) {
            const uint64_t u = (uint64_t)uu;
            Rng r(seed, 0x200000000ull + u);
            double x = raw[u] * scale;
            uint64_t d = (uint64_t)x + (r.unif() < x - std::floor(x) ? 1 : 0);
            if (d > 20000) d = 20000;
            uint64_t h = (uint64_t)(std::upper_bound(host_start.begin(), host_start.end(), (uint32_t)u) -
                                    host_start.begin()) - 1;
            const uint64_t hs = host_start[h], he = host_start[h + 1], hsz = he - hs;
            auto& row = rows[u];
            row.reserve(d + 16);
            for (int round = 0; round < 8 && row.size() < d; round++) {
                while (row.size() < d) {
                    double p = r.unif();
                    if (p < 0.70) {                               // run of consecutive ids near u in the host
                        uint64_t len = 1 + (uint64_t)(-std::log(1.0 - r.unif()) * 11.0);
                        int64_t off = (int64_t)std::floor(pareto(r, 1.0, (double)hsz, 1.5));
                        if (r.unif() < 0.5) off = -off;
                        int64_t st = (int64_t)u + off;
                        if (st < (int64_t)hs) st = (int64_t)hs;
                        for (uint64_t t = 0; t < len && row.size() < d + 8; t++) {
                            uint64_t v = (uint64_t)st + t;
                            if (v >= he) break;
                            row.push_back((uint32_t)v);
                        }
                    } else if (p < 0.95) {                        // short-gap link inside the host
                        int64_t off = (int64_t)std::floor(pareto(r, 1.0, (double)hsz, 1.2));
                        if (r.unif() < 0.5) off = -off;
                        int64_t v = (int64_t)u + off;
                        if (v < (int64_t)hs) v = (int64_t)hs + (int64_t)r.below(hsz);
                        if (v >= (int64_t)he) v = (int64_t)hs + (int64_t)r.below(hsz);
                        row.push_back((uint32_t)v);
                    } else {                                      // inter-host link, preferential host choice
                        uint64_t t = (uint64_t)(pareto(r, 1.0, (double)H, 1.0)) - 1;
                        if (t >= H) t = H - 1;
                        uint64_t ts = host_start[t], tsz = host_start[t + 1] - ts;
                        uint64_t v = r.unif() < 0.5 ? ts : ts + r.below(tsz);
                        row.push_back((uint32_t)v);
                    }
                }
                std::sort(row.begin(), row.end());            // duplicates do not count towards the degree
                row.erase(std::unique(row.begin(), row.end()), row.end());
                if (hsz <= d) break;                          // host too small to hold d distinct targets
            }
        }
        Graph* g = new Graph();
        rows_to_csr(n, rows, *g, false);
        if (relabel) bfs_relabel(*g);
        return (syn_graph*)g;
    } catch (...) {
        return nullptr;
    }
}

// Social digraph (twitter-2010 shape):
//  * out-degree power-law (alpha 1.9) in [1, max_deg], ~5% zero, rescaled to mean_deg;
//  * communities = contiguous id ranges, sizes power-law (alpha 1.7) in [20, 5e4];
//  * ~60% of arcs uniform inside the community, ~40% to globally preferential targets (density ~ x^(-2/3) over a
//    fixed random relabelling of ids, i.e. a power-law in-degree);
//  * then BFS-order relabelling.
syn_graph* syn_social(uint64_t n, double mean_deg, uint64_t max_deg, uint64_t seed, int relabel) {
    try {
        std::vector<uint32_t> com_start;
        {
            Rng r(seed, 0xC0ull);
            uint64_t p = 0;
            while (p < n) {
                com_start.push_back((uint32_t)p);
                p += (uint64_t)pareto(r, 20.0, 5e4, 1.7);
            }
            com_start.push_back((uint32_t)n);
        }
        std::vector<double> raw(n);
        double sum = 0.0;
#pragma omp parallel for reduction(+ : sum) schedule(static)
        for (int64_t u = 0; u < (int64_t)n; u++) {
            Rng r(seed, 0x100000000ull + (uint64_t)u);
            raw[u] = r.unif() < 0.05 ? 0.0 : pareto(r, 1.0, (double)max_deg, 1.9);
            sum += raw[u];
        }
        const double scale = mean_deg * (double)n / sum;
        // popularity permutation: rank -> id (a multiplicative hash permutation of [0, n) via cycle walking)
        const uint64_t mult = 0x9E3779B1ull | 1ull;
        uint64_t P = 1;
        while (P < n) P <<= 1;
        auto perm = [&](uint64_t x) {
            do { x = (x * mult + 0x7F4A7C15ull) & (P - 1); } while (x >= n);
            return x;
        };
        std::vector<std::vector<uint32_t>> rows(n);
#pragma omp parallel for schedule(dynamic, 64)
        for (int64_t uu = 0; uu < (int64_t)n; uu++) {
            const uint64_t u = (uint64_t)uu;
            Rng r(seed, 0x200000000ull + u);
            double x = raw[u] * scale;
            uint64_t d = (uint64_t)x + (r.unif() < x - std::floor(x) ? 1 : 0);
            if (d > max_deg) d = max_deg;
            if (d > n - 1) d = n - 1;
            uint64_t c = (uint64_t)(std::upper_bound(com_start.begin(), com_start.end(), (uint32_t)u) -
                                    com_start.begin()) - 1;
            const uint64_t cs = com_start[c], csz = com_start[c + 1] - cs;
            auto& row = rows[u];
            row.reserve(d);
            for (int round = 0; round < 8 && row.size() < d; round++) {
                while (row.size() < d) {
                    if (r.unif() < 0.6 && csz > 1) row.push_back((uint32_t)(cs + r.below(csz)));
                    else {
                        double q = r.unif();
                        uint64_t rank = (uint64_t)(std::pow(q, 3.0) * (double)n);
                        if (rank >= n) rank = n - 1;
                        row.push_back((uint32_t)perm(rank));
                    }
                }
                std::sort(row.begin(), row.end());            // duplicates do not count towards the degree
                row.erase(std::unique(row.begin(), row.end()), row.end());
            }
        }
        Graph* g = new Graph();
        rows_to_csr(n, rows, *g, false);
        if (relabel) bfs_relabel(*g);
        return (syn_graph*)g;
    } catch (...) {
        return nullptr;
    }
}

}  // extern "C"
