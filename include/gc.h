/*
 * gc.h -- C ABI of the B200-native independent-set graph colouring library
 * (libgc.so, built from paper_conf_ipps_osamatybo19_b200/csrc for sm_100a).
 *
 * Method: Osama, Truong, Yang, Buluc, Owens, "Graph Coloring on the GPU",
 * IPDPS-W 2019.  "P:L<n>" cites PAPER.md line n; "Alg.5 L<k>"
 * cites line k of the paper's Algorithm 5.  R<n> are the readings of silent
 * or garbled passages listed in DESIGN.md ("Readings").
 *
 * Problem: given an undirected graph G = (V, E), return
 * C : V -> N with C(v) != C(u) for every (v, u) in E.
 *
 * Conventions shared by every entry point
 *   - Graphs are CSR: row_offsets int64[n+1] (monotone,
 *     row_offsets[0] == 0, row_offsets[n] == nnz), col_indices uint32[nnz]
 *     (every value < n).  The adjacency must be symmetric and free of
 *     self-loops (the paper symmetrises and removes loops);
 *     duplicate entries and unsorted rows are accepted (adjacency is a set).
 *   - Pointers may be host or device memory; the library detects which with
 *     cudaPointerGetAttributes.  Host memory may be pageable or pinned.
 *   - Every function returns a negative gc_status on failure and never aborts
 *     the process; gc_last_error() then holds a thread-local message.
 *   - Work runs on the handle's stream (gc_set_stream; default: the legacy
 *     default stream) on the CUDA device that was current at create time.
 *     gc_color* return after the result is complete (they synchronise the
 *     stream once at the end, and once per batch of rounds).
 *   - A handle is not thread-safe; distinct handles are independent.
 *   - There is no CPU fallback: without a usable sm_100 device every call
 *     fails with GC_ERR_CUDA.
 */
#ifndef GC_H
#define GC_H

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

#define GC_ABI_VERSION 1

/* ----------------------------------------------------------- status codes */
typedef enum gc_status {
    GC_OK = 0,
    GC_ERR_INVALID_ARG = -1,   /* null pointer, n < 0, non-monotone offsets,
                                  col >= n, nnz mismatch, bad variant/options */
    GC_ERR_SELF_LOOP = -2,     /* a self-loop never terminates (Alg.5 L29-34
                                  with u = v fails both strict tests; R7) */
    GC_ERR_NOT_SYMMETRIC = -3, /* gc_create_csr: with GC_VALIDATE; gc_color: Alg.2 / Alg.4 in COUNT
                                  mode (and the partitioned COUNT rounds) when the adjacency SETS
                                  are not symmetric (the other variants fall back to the witness /
                                  sweep kernels instead) */
    GC_ERR_TOO_LARGE = -4,     /* n >= 2^32, or colours would pass INT32_MAX */
    GC_ERR_CUDA = -5,          /* CUDA runtime error / no usable device */
    GC_ERR_NCCL = -6,          /* NCCL error in the distributed path */
    GC_ERR_OOM = -7            /* device allocation failed */
} gc_status;

/* ------------------------------------------------------------- variants */
/* GC_MAXMIN: Alg.5 -- per round k every uncoloured vertex that
 *   is the strict local maximum of its weight among uncoloured neighbours gets
 *   colour 2k, the strict local minimum gets 2k+1 (a vertex with no
 *   uncoloured neighbour is both and takes 2k+1, Alg.5 L37-42, R9).
 * GC_LUBY_MIS: Alg.2 with the Alg.3 maximal-independent-set
 *   inner loop: colour c is a maximal independent set of the
 *   still-uncoloured vertices, built by repeated local-max selection with
 *   fixed weights (R10).  Colours are 0..n_colors-1.
 * GC_MULTIHASH(h): h independent weight functions per round (R8): vertex v
 *   takes colour 2(kh+j) (max) or 2(kh+j)+1 (min) for the smallest hash j
 *   under which it is a local max or min.  GC_MULTIHASH(1) == GC_MAXMIN.
 *   1 <= h <= 16.
 * GC_IS_ALG2: Alg.2 as written, max-only IS: iteration k
 *   colours the uncoloured vertices heavier than every uncoloured neighbour
 *   with colour k.  COUNT mode only; single GPU.
 * GC_JP_ALG4: Alg.2 with Alg.4 (reading R15): the same
 *   frontiers, each frontier takes ONE colour, the smallest colour not used by
 *   any coloured neighbour of the frontier (GraphBLAS Jones-Plassmann).
 *   COUNT mode only; single GPU.
 * GC_HASH_IS(t): the paper's Hash IS (Alg.6) made
 *   deterministic (R16-R20): per round every uncoloured vertex
 *   proposes the heaviest and the lightest of itself and its uncoloured
 *   neighbours; a proposed vertex reuses the smallest colour used so far that
 *   is not in its prohibited table of t colours (0 <= t <= 64), else takes a
 *   new colour (2k max / 2k+1 min); conflicts reset the lighter endpoint (or
 *   the new vertex, against an older colour).  Own per-round kernels
 *   (gc_stats.mode_used = GC_MODE_SWEEP, options.mode ignored); single GPU. */
#define GC_MAXMIN 0
#define GC_LUBY_MIS 1
#define GC_MULTIHASH(h) (2 | ((h) << 8))
#define GC_IS_ALG2 3
#define GC_JP_ALG4 4
#define GC_HASH_IS(t) (5 | ((t) << 8))
#define GC_HASH_TABLE_MAX 64
#define GC_VARIANT_KIND(v) ((v) & 0xFF)
#define GC_VARIANT_HASHES(v) (((v) >> 8) & 0xFF)
/* GC_LDF(v): largest-degree-first priorities (PAPER.md:1090-1098,
 *   reading R21): the weight of v becomes the pair (deg(v), p(v)), compared
 *   lexicographically (the larger degree wins, the seeded weight breaks
 *   ties; deg = number of distinct neighbours).  Applies to GC_MAXMIN,
 *   GC_LUBY_MIS, GC_IS_ALG2 and GC_JP_ALG4; COUNT mode, single GPU.  An
 *   asymmetric adjacency returns GC_ERR_NOT_SYMMETRIC (no fallback). */
#define GC_LDF(v) ((v) | (1 << 16))
#define GC_VARIANT_LDF(v) (((v) >> 16) & 1)

/* ---------------------------------------------------------------- flags */
#define GC_BORROW_DEVICE (1u << 0) /* create: adopt device CSR pointers without
                                      copying; caller keeps them alive */
#define GC_VALIDATE (1u << 1)      /* create: also check symmetry, O(m log d) */
#define GC_COMPACT (1u << 2)       /* color: renumber raw colours to
                                      0..n_colors-1 in increasing order (R12) */
#define GC_OUT_LOCAL_SLICE (1u << 3) /* distributed color: colors_out holds only
                                        the owned range [v_begin, v_end) */
#define GC_PROFILE (1u << 4)       /* color: time every sweep-kernel launch with
                                      CUDA events on the handle's stream and count
                                      visits (fills gc_stats.kernel_*; adds a
                                      little overhead, so keep it out of timed runs) */

/* Sweep strategy (gc_options.mode).  All modes return identical colours. */
#define GC_MODE_AUTO 0   /* max-min and multi-hash: SWEEP if max degree <= 8
                            and n >= 2^20 (large meshes), else COUNT;
                            Luby-MIS: COUNT */
#define GC_MODE_SWEEP 1  /* every round re-scans each uncoloured vertex's row
                            with early exit (the paper's ComputeOp shape) */
#define GC_MODE_EVENT 2  /* work-efficient: per-vertex witnesses + resume
                            cursors; only neighbours of newly coloured
                            vertices are re-evaluated; all
                            rounds in one persistent cooperative kernel */
#define GC_MODE_EVENT_MULTI 3 /* the same method, 4 kernel launches per round */
#define GC_MODE_COUNT 4  /* work-efficient: per-vertex counts of uncoloured
                            larger / smaller neighbours; each row is walked
                            once, when its vertex is coloured (one atomic per
                            entry); one persistent kernel, one grid barrier
                            per round.  Luby-MIS: the same
                            colouring (first-fit greedy in decreasing weight
                            order, R10) as a Jones-Plassmann wavefront over
                            predecessor counts; a vertex's colour is the mex
                            of its predecessors' colours;
                            gc_stats.rounds / inner_iterations are then the
                            wavefront depth, not Alg.3's iteration count.
                            Multi-hash: H count pairs per vertex, the
                            decision of a vertex kept as its first free
                            (round, j, side) */

typedef struct gc_graph gc_graph;

/* Options for gc_color_ex.  Zero-initialise, then set struct_size. */
typedef struct gc_options {
    uint32_t struct_size;     /* sizeof(gc_options) */
    int32_t variant;          /* GC_MAXMIN / GC_LUBY_MIS / GC_MULTIHASH(h) */
    uint64_t seed;            /* weight seed (R1) */
    uint32_t flags;           /* GC_COMPACT, GC_OUT_LOCAL_SLICE */
    int32_t mode;             /* GC_MODE_* */
    int32_t batch_rounds;     /* rounds enqueued per host check; 0 = adaptive */
    int32_t thread_deg_max;   /* sweep: rows <= this scanned by one thread (0=default) */
    int32_t hub_deg_min;      /* sweep: rows >= this scanned by a CTA (0=default) */
    int32_t reserved[7];
} gc_options;

/* Statistics filled by gc_color_ex (optional). */
typedef struct gc_stats {
    uint32_t struct_size;     /* sizeof(gc_stats) */
    int32_t mode_used;        /* GC_MODE_SWEEP, GC_MODE_EVENT, GC_MODE_EVENT_MULTI or GC_MODE_COUNT */
    int64_t rounds;           /* R: rounds (max-min / multi-hash) or colours (Luby) */
    int64_t inner_iterations; /* Luby: Alg.3 do-while iterations; else == rounds */
    int64_t n_colors;         /* distinct colours */
    int64_t launches;         /* kernels launched by this call */
    double ms;                /* device time of the call (CUDA events) */
    int64_t *frontier_sizes;  /* optional caller buffer: N_k per round (not written for
                                 Luby-MIS and GC_HASH_IS) */
    int64_t frontier_cap;     /* its capacity */
    /* GC_PROFILE only.  Kernel classes: [0] the per-round sweep kernel (the
     * hot loop), [1] the hub (CTA-per-row) kernel, [2] everything else.
     * kernel_bytes = algorithmic HBM bytes of that class (DESIGN.md
     * "Algorithmic bytes"); visits = neighbour entries examined. */
    double kernel_ms[4];
    int64_t kernel_launches[4];
    int64_t kernel_bytes[4];
    int64_t visits;
    /* GC_PROFILE only, optional caller buffers: the duration of every timed
     * launch in launch order (us), and per round 16 values (event mode:
     * |D_k| evaluated, |I_k| coloured, long scans, long-row notify items,
     * the persistent kernel's P1 / P1b+P2 / P3 phase times in ns, -, then
     * the longest per-block work time of P1 / P1b / P2 / P3 in ns;
     * sweep mode: N_k, 0...). */
    float *launch_us;
    int64_t launch_cap;
    int64_t *round_stats;
    int64_t round_stats_cap;  /* in rounds */
} gc_stats;

/* ------------------------------------------------------------ lifecycle */
/* Create a graph handle from CSR arrays (host or device).  The arrays are
 * copied into device memory owned by the handle (the caller may free its
 * copies on return) unless GC_BORROW_DEVICE is set and both arrays are device
 * pointers.  Checks: n >= 0, n < 2^32, nnz == row_offsets[n], monotone
 * offsets, col < n, no self-loops (GC_ERR_SELF_LOOP); with GC_VALIDATE also
 * symmetry (GC_ERR_NOT_SYMMETRIC).  On success *out receives the handle. */
int gc_create_csr(int64_t n, int64_t nnz, const int64_t *row_offsets,
                  const uint32_t *col_indices, uint32_t flags, gc_graph **out);

/* Colour the graph: Alg.1 driven by the variant's independent
 * set rule.  colors_out: caller-allocated int32[n] (host or device) receives
 * raw colours (or compacted ones with GC_COMPACT via gc_color_ex).  Returns
 * n_colors >= 1 (0 iff n == 0), or a negative gc_status.  The result is a
 * pure function of (adjacency sets, seed, variant): independent of row order,
 * duplicates, launch configuration, mode and batch size. */
int64_t gc_color(gc_graph *g, uint64_t seed, int32_t variant, int32_t *colors_out);

/* As gc_color with explicit options and optional statistics (stats may be
 * NULL).  opts must not be NULL and opts->struct_size must be set. */
int64_t gc_color_ex(gc_graph *g, const gc_options *opts, int32_t *colors_out,
                    gc_stats *stats);

/* Use this cudaStream_t for all subsequent work of the handle. */
int gc_set_stream(gc_graph *g, void *cuda_stream);

/* Release the handle and its device memory.  NULL-safe. */
void gc_destroy(gc_graph *g);

/* Thread-local description of the last failure ("" if none). */
const char *gc_last_error(void);

/* ---------------------------------------------------------- components */
/* a0: the vertex weights (Alg.5 L7 "generateRandomNumbers"; R1):
 * out[i] = p_j(v_begin + i) for i < count.  out is host or device. */
int gc_priorities(uint64_t seed, int32_t j, int64_t v_begin, int64_t count, uint32_t *out);

/* Number of distinct values in colors[0..n) (host or device), >= 0. */
int64_t gc_count_colors(const int32_t *colors, int64_t n);

/* Library build information (e.g. "gc 1 sm_100a cuda 12.9"). */
const char *gc_version(void);

/* Memory: device and pinned-host blocks released by gc_destroy are kept in a
 * per-device cache and reused by later handles (creating a handle then maps
 * no new pages; a cudaMalloc that fails first returns the cache to the
 * driver).  gc_trim returns every cached block to the driver now; GC_OK.
 * Setting GC_NO_CACHE=1 in the environment disables the cache. */
int gc_trim(void);

/* ---------------------------------------------------- distributed (1D) */
/* Create a rank's share of a graph partitioned by contiguous vertex ranges:
 * this rank owns rows [v_begin, v_end) of an n_global-vertex graph.
 * row_offsets_local: int64[v_end - v_begin + 1] starting at 0;
 * col_indices_global: uint32[nnz_local] holding GLOBAL vertex ids.
 * nccl_unique_id: 128 bytes from ncclGetUniqueId on rank 0, broadcast by the
 * caller (e.g. over a torch process group).  Collective over `world` ranks.
 * gc_color / gc_color_ex on the handle are then collective too: every rank
 * calls them with the same seed/variant; colors_out receives the full n_global
 * colours (or only the owned slice with GC_OUT_LOCAL_SLICE).  Results equal
 * the single-GPU colouring bit for bit.  Supported variants: GC_MAXMIN and
 * GC_MULTIHASH(h). */
int gc_create_csr_dist(int64_t n_global, int64_t v_begin, int64_t v_end,
                       int64_t nnz_local, const int64_t *row_offsets_local,
                       const uint32_t *col_indices_global,
                       const void *nccl_unique_id, int rank, int world,
                       uint32_t flags, gc_graph **out);

/* Fill 128 bytes with a fresh NCCL unique id (call on rank 0 only). */
int gc_nccl_unique_id(void *out128);

/* The partitioned algorithm of gc_create_csr_dist run on ONE GPU: the graph
 * (same arguments as gc_create_csr) is split into `parts` equal vertex ranges,
 * each with its own colour replica, exchanged every round by device copies
 * instead of NCCL.  gc_color on the handle returns exactly the single-GPU
 * colouring; this is how the partition / exchange logic is tested on one GPU. */
int gc_create_csr_loopback(int64_t n, int64_t nnz, const int64_t *row_offsets,
                           const uint32_t *col_indices, int parts, uint32_t flags,
                           gc_graph **out);

#ifdef __cplusplus
}
#endif

#endif /* GC_H */
