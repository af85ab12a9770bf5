/*
 * gcgt.h — C ABI of the B200-native GCGT hot path (Sha, Li, Tan, "GPU-based Graph Traversal on Compressed
 * Graphs", SIGMOD '19).  Library: paper_conf_sigmod_shalt19_b200/libgcgt.so (sm_100a CUDA + host C++).
 *
 * The boundary follows the paper's problem statement (§3.2, Fig. 3): the CPU compresses the
 * graph into the compressed graph representation (CGR), the CGR is moved to device memory without being
 * decompressed there, and the CPU issues traversal queries that run on the CGR.  Application outputs are
 * per-vertex labels (§6 :1137-1286, Fig. 7).  The exact bit layout is FORMAT.md (rules R1-R19).
 *
 * Conventions (every entry point):
 *  - Plain C types only; no C++ or torch types cross the boundary; no exception escapes.
 *  - Ownership: the caller owns every buffer it passes in or out.  The library owns gcgt_cgr / gcgt_graph
 *    objects until gcgt_cgr_free / gcgt_unload.
 *  - Errors: a gcgt_status is returned; on anything but GCGT_OK, gcgt_last_error() returns a thread-local
 *    message.  Inputs are validated before any allocation; on error no output buffer is partially trusted.
 *  - Synchronisation: every call is synchronous with respect to the graph's stream on return (outputs are
 *    complete and visible to the host or the device).
 *  - Vertex ids are uint32 (n <= 2^32 - 1); bit offsets and arc counts are uint64.
 *  - There is no CPU fallback: gcgt_load / gcgt_bfs / gcgt_cc / gcgt_bc fail with GCGT_ECUDA when no CUDA
 *    device is usable.
 */
#ifndef GCGT_H
#define GCGT_H

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

typedef enum {
    GCGT_OK = 0,
    GCGT_EINVAL = -1,     /* bad argument / parameter (e.g. min_interval_len == 1, zeta_k outside 1..5)      */
    GCGT_EUNSORTED = -2,  /* a CSR row is not strictly increasing (FORMAT.md R6)                              */
    GCGT_ERANGE = -3,     /* a column id or a source >= n                                                     */
    GCGT_ESEGLEN = -4,    /* a residual segment cannot hold even one residual (FORMAT.md R19)                */
    GCGT_ENOMEM = -5,     /* host or device allocation failed                                                 */
    GCGT_ECUDA = -6,      /* CUDA runtime error, or no usable device                                          */
    GCGT_ERESERVED = -7,  /* (unused)                                                                          */
    GCGT_EFORMAT = -8     /* corrupt or inconsistent CGR (file or view)                                        */
} gcgt_status;

/* Input graph in CSR (Fig. 1): out-arcs of u are cols[row_offsets[u] .. row_offsets[u+1]).
 * Host memory, caller-owned.  m = row_offsets[n].  Rows must be strictly increasing with ids < n. */
typedef struct {
    uint64_t n;
    const uint64_t* row_offsets; /* n + 1 entries */
    const uint32_t* cols;        /* row_offsets[n] entries */
} gcgt_csr;

/* CGR parameters (Table 2; App. D sweeps them). */
typedef struct {
    uint32_t min_interval_len;     /* 0 = no intervals ("inf", Fig. 12); otherwise >= 2.  Paper default 4.          */
    uint32_t residual_segment_len; /* residual segment length in BYTES (FORMAT.md R15); 0 = unsegmented ("inf").
                                      Paper default 32.                                                               */
    uint32_t zeta_k;               /* 1 = gamma code, 2..5 = the paper's zeta_k (App. B, Table 3).  Paper default 3. */
} gcgt_params;

/* Per-call statistics (optional; pass NULL to skip). */
typedef struct {
    uint32_t iterations;        /* BFS: levels expanded; CC: hook iterations; BC: sources processed             */
    uint32_t reserved;
    uint64_t vertices_expanded; /* frontier vertices whose CGR record was decoded (summed over passes)         */
    uint64_t arcs_decoded;      /* neighbour ids produced by decoding (summed over passes)                     */
    uint64_t cgr_bits_decoded;  /* CGR bits of the records decoded (algorithmic CGR traffic)     */
    double device_ms;           /* device time of the call (CUDA events on the graph's stream)                 */
    double kernel_ms;           /* with gcgt_profile(g, 1): summed CUDA-event time of the call's dominant kernel
                                   (BFS/BC: frontier expansion; CC: hooking), else 0                              */
    uint64_t kernel_launches;   /* launches of that kernel in the call (0 unless profiling)                      */
    uint64_t launches;          /* all library kernel launches of the call                                       */
} gcgt_stats;

typedef struct gcgt_cgr gcgt_cgr;     /* host CGR: canonical bytes + bit_offsets + params; library-owned     */
typedef struct gcgt_graph gcgt_graph; /* device-resident CGR and work buffers; library-owned                  */

/* ---- Graph Compression Module (CPU; §3.1 :353-411, App. C :2097-2112, §5.2 :1092-1136, Fig. 3) ------------------
 * gcgt_encode: CSR -> CGR, bit-exact with FORMAT.md.  Multi-threaded (OpenMP).  *out receives a new object.
 * Errors: EINVAL (params), EUNSORTED / ERANGE (input rows), ESEGLEN (segment too short), ENOMEM. */
gcgt_status gcgt_encode(const gcgt_csr* csr, const gcgt_params* params, gcgt_cgr** out);

/* Encodes the TRANSPOSE of csr (row v = sorted in-neighbours of v), for gcgt_load_opts.in_cgr.  Same errors. */
gcgt_status gcgt_encode_transpose(const gcgt_csr* csr, const gcgt_params* params, gcgt_cgr** out);

/* Vertex-range slices (graphs too large to hold as one CSR, e.g. C5 = R-MAT scale 29): gcgt_encode_slice encodes
 * rows 0..rows->n-1 of a caller CSR as the records of vertices first .. first + rows->n - 1 of a graph with n_total
 * vertices (column ids < n_total); the bytes equal bits [bit_offsets[first], bit_offsets[first + rows->n]) of the
 * whole graph's CGR (records are self-contained, R2), bit offsets re-based to 0.  gcgt_cgr_concat appends
 * consecutive slices into one CGR (EINVAL unless consecutive, same parameters and n_total).  gcgt_load of a slice
 * loads exactly its vertex range as a partitioned graph (first and first + rows->n on 32-vertex words, or the end). */
gcgt_status gcgt_encode_slice(const gcgt_csr* rows, uint64_t first, uint64_t n_total, const gcgt_params* params,
                              gcgt_cgr** out);
gcgt_status gcgt_cgr_concat(const gcgt_cgr* const* parts, uint32_t k, gcgt_cgr** out);
gcgt_status gcgt_cgr_slice_info(const gcgt_cgr* cgr, uint64_t* first, uint64_t* n_total);

/* Read-only view of a CGR: bytes (ceil(nbits/8), MSB-first, R1), nbits, bit_offsets (n + 1 entries, R2),
 * n, params.  Pointers stay valid until gcgt_cgr_free.  Any output pointer may be NULL. */
gcgt_status gcgt_cgr_view(const gcgt_cgr* cgr, const uint8_t** bytes, uint64_t* nbits,
                          const uint64_t** bit_offsets, uint64_t* n, gcgt_params* params);

/* Builds a CGR object by copying caller arrays (e.g. a CGR produced elsewhere).  Checks bit_offsets is
 * non-decreasing with bit_offsets[n] == nbits; returns EFORMAT otherwise. */
gcgt_status gcgt_cgr_from_arrays(uint64_t n, const uint8_t* bytes, uint64_t nbits, const uint64_t* bit_offsets,
                                 const gcgt_params* params, gcgt_cgr** out);

/* Checkpoint / resume of the offline artefact (the CGR is the only persistent state, Fig. 3 :438-454). */
gcgt_status gcgt_cgr_save(const gcgt_cgr* cgr, const char* path);
gcgt_status gcgt_cgr_open(const char* path, gcgt_cgr** out);
void gcgt_cgr_free(gcgt_cgr* cgr);

/* Prepares a whole CGR for repeated loads (a query service that reloads the graph): builds the derived load tables
 * now -- the compact bit offsets and the interval checkpoint table, otherwise built on
 * the first gcgt_load and kept with the CGR -- and page-locks the CGR's host arrays (cudaHostRegister, portable), so
 * that each later gcgt_load is host-to-device DMA plus the device byte swap.  Idempotent; the registration is
 * released by gcgt_cgr_free.  ECUDA if page-locking fails (nothing is left registered by the failing call's array). */
gcgt_status gcgt_cgr_pin(gcgt_cgr* cgr);

/* ---- Device residency (§3.2 :469-479: "directly move the compressed adjacency lists to GPUs") -------------------- */
typedef struct {
    int device;        /* CUDA device ordinal                                                                       */
    void* stream;      /* cudaStream_t to run on (cudaStreamLegacy = (void*)1 for the legacy default stream); NULL = a
                          library-created non-blocking stream                                                       */
    int rank, nranks;  /* 1-D vertex-range partition (multi-GPU).  nranks <= 1: single GPU (rank ignored)           */
    void* reserved;    /* must be NULL (the collectives of the partitioned steps run in the caller)                  */
    const gcgt_cgr* in_cgr; /* CGR of the TRANSPOSE (in-arcs, e.g. from gcgt_encode_transpose) for the bottom-up
                               BFS step; NULL = none (top-down only unless `symmetric`).  Same n and params.      */
    int symmetric;     /* 1: every arc u->v has v->u, so the out-CGR doubles as the in-CGR (R-MAT configs)           */
    int direction_optimizing; /* 0: top-down only; 1: switch top-down <-> bottom-up per level when an in-CGR exists */
    int host_resident; /* 1: keep the CGR words (and the in-CGR's) in pinned, mapped HOST memory owned by the graph and
                          decode them over the host link (zero copy; §8 f4, the out-of-core motivation PAPER.md:93-120,
                          :474-479); bit offsets, bitmaps and outputs stay in device memory.  Results are identical;
                          only the bandwidth differs.  0: the CGR is copied to HBM (default).                      */
} gcgt_load_opts;

/* Copies the CGR (bytes + bit_offsets) to the device and allocates the traversal work buffers.  With nranks > 1
 * each rank keeps only the records of its owned vertex range (balanced by CGR bits; records are self-contained,
 * so slicing is a bit copy) plus replicated n-bit bitmaps.  opts may be NULL (device 0, own stream). */
gcgt_status gcgt_load(const gcgt_cgr* cgr, const gcgt_load_opts* opts, gcgt_graph** out);

/* Uncompressed baseline (§8 f3; the paper's GPUCSR comparison, Fig. 8 :1571-1578): copies a
 * plain CSR (host, caller-owned; rows need not be sorted; ids < n < 2^32) to the device.  gcgt_bfs on the result
 * runs the same frontier / filter / contraction / direction machinery as the CGR path with expansion reading
 * col[] instead of decoding, so the time ratio is the decoding overhead.  With direction_optimizing the bottom-up
 * in-lists are the transpose (built on the host) or, when `symmetric`, the CSR itself; opts->in_cgr is ignored.
 * Single GPU only (nranks <= 1).  gcgt_cc / gcgt_bc / gcgt_dist_* return EINVAL on such a graph.
 * stats->cgr_bits_decoded counts 32 bits per col[] entry read.  Errors: EINVAL, ERANGE (id >= n), ENOMEM, ECUDA. */
gcgt_status gcgt_load_csr(const gcgt_csr* csr, const gcgt_load_opts* opts, gcgt_graph** out);
void gcgt_unload(gcgt_graph* g);

/* Enables (1) / disables (0) per-launch CUDA-event timing of the dominant kernel (fills gcgt_stats.kernel_ms).
 * Adds one event pair per launch, read at the call's existing host syncs (the BFS level loop stays asynchronous);
 * results are unchanged.  2 = also per-level spans (gcgt_profile_spans): the BFS level loop then waits per level. */
gcgt_status gcgt_profile(gcgt_graph* g, int enable);

/* With span profiling on (gcgt_profile(g, 2)), the last gcgt_bfs call's device time split into spans (ms): [0]
 * top-down expansion kernel(s), [1] hub segments / interval chunks, [2] bottom-up kernel, [3] contraction +
 * direction choice.  count <= 4. */
gcgt_status gcgt_profile_spans(const gcgt_graph* g, double* ms, int count);

/* Owned vertex range [*lo, *hi) of this rank (whole [0, n) on a single GPU). */
gcgt_status gcgt_graph_range(const gcgt_graph* g, uint64_t* lo, uint64_t* hi);

/* ---- Traversal queries (§4-§6; Fig. 7) ------------------------------------------------------------------------ */
/* Output placement flag for the query calls below. */
#define GCGT_OUT_HOST 0   /* output pointer is host memory (pageable or pinned); the library copies D2H       */
#define GCGT_OUT_DEVICE 1 /* output pointer is device memory on the graph's device                             */

/* BFS from `source` over out-arcs (Fig. 7(b)).  levels[v] = hop distance, -1 if unreached; n entries.
 * With an in-CGR (or `symmetric`) and direction_optimizing, large levels run bottom-up: every unvisited vertex
 * decodes its in-record until the first frontier parent (intervals tested as frontier-bitmap ranges).
 * Errors: ERANGE (source >= n), ECUDA. */
gcgt_status gcgt_bfs(gcgt_graph* g, uint32_t source, int32_t* levels, int out_placement, gcgt_stats* stats);

/* Weakly connected components (Fig. 7(c): hooking + pointer jumping, Soman et al. [42]).  labels[v] = the
 * minimum vertex id in v's component (every arc joins both endpoints); n entries. */
gcgt_status gcgt_cc(gcgt_graph* g, uint32_t* labels, int out_placement, gcgt_stats* stats);

/* Betweenness centrality from k sources (host array; duplicates counted), Brandes' dependency accumulation
 * (Fig. 7(d), §6 :1272-1284): bc[v] = sum_s delta_s(v), v != s; unnormalised, fp64; n entries.
 * Errors: ERANGE (a source >= n). */
gcgt_status gcgt_bc(gcgt_graph* g, const uint32_t* sources, uint32_t k, double* bc, int out_placement,
                    gcgt_stats* stats);

/* ---- Partitioned multi-GPU steps (§8 e; driver: paper_conf_sigmod_shalt19_b200/dist.py) -----------------------
 * A graph loaded with nranks > 1 holds only its owned vertex range [lo, hi) (gcgt_graph_range; boundaries on
 * 32-vertex words, balanced by CGR bits): the out-records of the owned vertices and, with in_cgr / symmetric, their
 * in-records.  The caller runs the collectives between the steps (e.g. NCCL through torch.distributed).  Every
 * bitmap crossing this boundary is a DEVICE array of ceil(n/32) uint32 words (bit v%32 of word v/32); an owned slice
 * is words [lo/32, ceil(hi/32)).  gcgt_bfs / gcgt_cc / gcgt_bc refuse partitioned graphs.
 * The steps are ENQUEUED on the graph's stream and return without waiting (the caller's collectives must run on that
 * stream or after gcgt_sync), except gcgt_dist_bfs_absorb and gcgt_dist_cc_hook, which return a count to the host:
 * one host synchronisation per BFS level and per CC round.  BFS level d:
 *   top-down (bottom_up = 0):
 *     gcgt_dist_bfs_expand : decode the owned frontier's records, claim unvisited targets into `cand` (full bitmap,
 *                            zeroed by the call)                                          [expansion + filter]
 *     (caller) all-to-all  : slice q of every rank's cand goes to rank q
 *     gcgt_dist_bfs_commit : fslice = OR(recv[0..nparts)) & ~visited; levels of the new owned vertices = d + 1
 *   bottom-up (bottom_up = 1; needs the in-records):
 *     gcgt_dist_bfs_expand : every owned unvisited vertex scans its in-record against the replicated frontier until
 *                            the first parent; finds are written to the owned slice `fslice` (no exchange needed)
 *     gcgt_dist_bfs_commit : with nparts = 0, keep = 1: fslice &= ~visited, levels = d + 1
 *   both:
 *     (caller) all-gather  : the owned fslices form the global next frontier
 *     gcgt_dist_bfs_absorb : frontier := gathered bitmap; visited |= frontier; *count = its size (identical on every
 *                            rank, so termination needs no extra collective)
 * gcgt_dist_bfs_levels copies the owned levels out.
 * CC: parent is a caller-owned device array of n uint32 replicated on every rank; per round
 *   gcgt_dist_cc_hook   hook the owned vertices' arcs (no path halving: hooks are the only writes to parent);
 *                       *hooks = successful hooks (host; the call waits); the first min(hooks, cap) hooks are also
 *                       written to `pairs` (device, 2 uint32 per hook: index hi, new parent lo < hi)
 *   exchange            all-reduce(MIN) of parent — or, when every rank's hooks fit cap, the pair lists
 *                       (all-gather) merged with gcgt_dist_cc_merge: parent[hi] = min(parent[hi], lo)
 *   gcgt_dist_cc_jump   pointer jumping
 *   and stop when no rank hooked.  Both exchanges leave identical parent arrays on every rank. */
gcgt_status gcgt_dist_bfs_begin(gcgt_graph* g, uint32_t source);
gcgt_status gcgt_dist_bfs_expand(gcgt_graph* g, uint32_t level, uint32_t* cand, uint32_t* fslice, int bottom_up);
gcgt_status gcgt_dist_bfs_commit(gcgt_graph* g, uint32_t level, const uint32_t* recv, uint32_t nparts,
                                 uint32_t* fslice, int keep);
gcgt_status gcgt_dist_bfs_absorb(gcgt_graph* g, const uint32_t* frontier, uint64_t* count);
gcgt_status gcgt_dist_bfs_levels(gcgt_graph* g, int32_t* levels_owned, int out_placement);
gcgt_status gcgt_dist_cc_hook(gcgt_graph* g, uint32_t* parent, uint32_t* pairs, uint64_t cap, uint64_t* hooks);
gcgt_status gcgt_dist_cc_merge(gcgt_graph* g, uint32_t* parent, const uint32_t* pairs, uint64_t npairs);
gcgt_status gcgt_dist_cc_jump(gcgt_graph* g, uint32_t* parent);

/* Waits for every step enqueued on the graph's stream (partitioned steps). */
gcgt_status gcgt_sync(gcgt_graph* g);

/* ---- Test hook (parity pin of the warp decoder against Fig. 5 / Ex. 5.1) ------------------
 * Runs the device warp-parallel decoder (Alg. 4 :901-919) on one warp over a caller bit array (host, MSB-first
 * bytes, R1): vals[0..count-1] receive the first `count` codewords decoded from bit 0; the FIRST window step over
 * `window` (16 or 32) lanes is traced: trace_pos / trace_flags (6 x 32 entries, row r = state after marking round
 * r, row 0 = initial; 0xFFFFFFFF = Fig. 5's 'x') and *rounds = number of rows written.  Uses device 0. */
gcgt_status gcgt_debug_warp_decode(const uint8_t* bytes, uint64_t nbits, uint32_t zeta_k, uint32_t window,
                                   uint64_t count, uint64_t* vals, uint32_t* trace_pos, uint32_t* trace_flags,
                                   uint32_t* rounds);

/* Thread-local message for the last non-OK status returned on this thread ("" if none). */
const char* gcgt_last_error(void);

/* Library / build identification string (compile target, e.g. "gcgt sm_100a"). */
const char* gcgt_version(void);

#ifdef __cplusplus
}
#endif
#endif /* GCGT_H */
