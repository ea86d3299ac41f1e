// gc_internal.cuh -- shared internals of libgc (the CUDA path).  Nothing here
// is shared with oracle/ (by rule: the oracle is an independent program).
#pragma once

#include <cuda_runtime.h>
#include <stdint.h>

#include <string>
#include <vector>

#include "../../include/gc.h"

#define GC_UNC 0xFFFFFFFFu  // "invalidColor" of Alg.5 L5
#define GC_MAX_HASHES 16

#include <nvtx3/nvToolsExt.h>  // header-only NVTX 3 (no link dependency; ranges cost ~nothing without a tool)

namespace gc {

// NVTX range for the lifetime of a scope (host side: shows each API call and
// phase on an Nsight timeline)
struct NvtxRange {
    explicit NvtxRange(const char *name) { nvtxRangePushA(name); }
    ~NvtxRange() { nvtxRangePop(); }
    NvtxRange(const NvtxRange &) = delete;
    NvtxRange &operator=(const NvtxRange &) = delete;
};


// ------------------------------------------------------------------ weights
// R1: p_j(v) = fmix32(v ^ K_j), K_j = fmix32(fold32(seed) +
// 0x9E3779B9 * (j + 1)).  fmix32 is MurmurHash3's 32-bit finaliser; it is a
// bijection on uint32 so weights never tie (R2).
__host__ __device__ __forceinline__ uint32_t weight_mix(uint32_t x) {
    x ^= x >> 16;
    x *= 0x85EBCA6Bu;
    x ^= x >> 13;
    x *= 0xC2B2AE35u;
    x ^= x >> 16;
    return x;
}

inline uint32_t weight_key(uint64_t seed, int j) {
    uint32_t folded = (uint32_t)(seed ^ (seed >> 32));
    return weight_mix(folded + 0x9E3779B9u * (uint32_t)(j + 1));
}

struct Keys {
    uint32_t k[GC_MAX_HASHES];
};

// ---------------------------------------------------------------- handle
struct Dist;  // distributed state (gc_dist.cu)

struct Scratch {
    // all device memory, sized for n (or n_local for the distributed path)
    uint32_t *C = nullptr;        // colours, GC_UNC = uncoloured
    uint32_t *F[2] = {nullptr, nullptr};  // frontiers (vertex ids)
    uint32_t *hub = nullptr;      // per-round hub work list / event: coloured list I_k
    uint32_t *Q = nullptr;        // event mode: long-scan queue
    uint32_t *Q2 = nullptr;       // event mode: long-row notify / long-scan segment queue
    uint32_t *Q3 = nullptr;       // persistent event mode: notify segment queue
    void *LS = nullptr;           // persistent event mode: long-scan slots (32 B each)
    uint32_t *M = nullptr;        // persistent event mode: round-start status bitmask
    uint32_t *S = nullptr;        // Luby inner-loop state / event stamps
    uint32_t *W = nullptr;        // event mode: witness pairs (2 per vertex)
    uint32_t *P = nullptr;        // event mode: resume cursors (2 per vertex)
    unsigned long long *ctr = nullptr;  // device counters (see gc_sweep.cu)
    int64_t *nk = nullptr;        // per-round frontier sizes (stats), cap nk_cap
    int64_t nk_cap = 0;
    int64_t *rstat = nullptr;     // PROF: 4 counters per round (cap nk_cap)
    uint32_t *bitmap = nullptr;   // colour-count bitmap
    unsigned long long *hist = nullptr;  // GC_PROFILE_HIST histograms (gc_persist.cu)
    int64_t bitmap_words = 0;
    int64_t *host_pinned = nullptr;  // pinned readback area
    // COUNT mode (gc_count.cu)
    unsigned long long *cnt = nullptr;   // (hi << 32) | lo uncoloured-neighbour counts (cnt_h per vertex)
    int cnt_h = 1;
    uint32_t *cnt32 = nullptr;           // packed (hi << 16) | lo counts (degree <= 65535)
    uint32_t *big = nullptr;             // vertices of degree > 65535
    uint32_t *big32 = nullptr;           // their per-side counts and flags
    int nbig = 0;                        // their number (-1: too many to pack)
    uint32_t *Z = nullptr;               // Zlo: round from which lo is free (freed second)
    void *SL = nullptr;                  // short-row items (16 B)
    void *WL = nullptr;                  // long-row segment items (16 B)
    uint32_t *hubs = nullptr;            // k_count: rows counted by blocks
    unsigned long long *cctr = nullptr;  // counters of the persistent count kernel
    int64_t sl_cap = 0, wl_cap = 0;
    uint32_t count_epoch = 0;            // COUNT colourings run (item round tags, gc_count.cu)
    uint32_t *cM = nullptr;              // COUNT mode: status bits (1 = uncoloured)
    uint32_t *crow = nullptr;            // COUNT mode: row of each counting chunk's first entry
    int64_t nch = 0;
    const int64_t *crow_ro = nullptr;    // ... of this CSR (row offsets, entries)
    int64_t crow_nnz = -1;
    uint32_t *deg = nullptr;             // LDF: row lengths (seed-independent)
    uint32_t *jslot = nullptr;           // JP (Luby-MIS in COUNT mode): mex slots of long rows
    uint32_t *jcr = nullptr;             // Alg.4: round colours + colour sets
    int64_t jcr_words = 0;
    int64_t jslot_cap = 0;
};

}  // namespace gc

struct gc_graph {
    int device = 0;
    int64_t n = 0;          // vertices owned (== n_global on one GPU)
    int64_t n_global = 0;
    int64_t v_begin = 0;    // owned range start
    int64_t nnz = 0;
    int64_t max_deg = 0;
    int64_t *ro = nullptr;  // device row offsets (local rows)
    uint32_t *ci = nullptr; // device column indices (global ids)
    bool owns_csr = true;
    cudaStream_t stream = 0;
    gc::Scratch s;
    gc::Dist *dist = nullptr;
    int sm_count = 148;
    bool count_unsafe = false;  // COUNT mode saw an asymmetric adjacency SET: use EVENT / SWEEP
    bool deduped = false;       // ro / ci were replaced by their deduplicated copy (gc_dedup.cu)
    bool rows_strict = false;   // every row strictly increasing (checked once, gc_dedup.cu)
};

namespace gc {

// A pair of CUDA events destroyed with the scope (every exit path).
struct EventPair {
    cudaEvent_t e0 = nullptr, e1 = nullptr;
    ~EventPair() {
        if (e0) cudaEventDestroy(e0);
        if (e1) cudaEventDestroy(e1);
    }
};

// ----------------------------------------------------------------- errors
void set_error(const std::string &msg);
int cuda_fail(cudaError_t e, const char *what);

// gc_alloc.cu: cached device / pinned-host allocations (free only when no
// pending device work uses the block)
cudaError_t dmalloc_raw(void **p, size_t bytes);
void dfree(void *p);
cudaError_t hmalloc_raw(void **p, size_t bytes);
void hfree(void *p);
template <class T>
inline cudaError_t dmalloc(T **p, size_t bytes) {
    return dmalloc_raw(reinterpret_cast<void **>(p), bytes);
}
template <class T>
inline cudaError_t hmalloc(T **p, size_t bytes) {
    return hmalloc_raw(reinterpret_cast<void **>(p), bytes);
}

#define GC_CUDA_TRY(expr)                                   \
    do {                                                    \
        cudaError_t _e = (expr);                            \
        if (_e != cudaSuccess) return gc::cuda_fail(_e, #expr); \
    } while (0)

bool is_device_ptr(const void *p);

// ------------------------------------------------------------- launchers
// GC_PROFILE accumulators (kernel classes: 0 sweep, 1 hub, 2 other)
struct Profile {
    bool on = false;
    double ms[4] = {0, 0, 0, 0};
    int64_t launches[4] = {0, 0, 0, 0};
    int64_t bytes[4] = {0, 0, 0, 0};
    int64_t visits = 0;
    std::vector<float> launch_us;   // every timed launch, in order
};

// Pool of CUDA events bracketing individual launches in profile mode.
struct EventTimer {
    std::vector<cudaEvent_t> ev;
    std::vector<int> cls;
    size_t used = 0;
    ~EventTimer();
    int begin(cudaStream_t st, int klass);   // records the start event
    int end(cudaStream_t st);                // records the matching stop event
    int drain(Profile *p);                   // after a stream sync: add durations
};

struct RunParams {
    Profile *prof = nullptr;
    int H = 1;
    Keys keys;
    int32_t thread_deg_max = 8;
    int32_t hub_deg_min = 4096;
    int32_t eval_big_min = 256;  // event mode: remaining scan length sent to a CTA
    int32_t batch_rounds = 0;
    int64_t max_rounds = 0;
    int ldf = 0;  // (degree, weight) priorities (R21), COUNT kernels only
};

struct RunResult {
    int64_t rounds = 0;
    int64_t inner = 0;
    int64_t launches = 0;
    int64_t max_color = -1;  // the largest colour, when the run computed it (else -1)
};

// One sweep round over a vertex range [v0, v0 + n_loc) (single GPU: v0 = 0).
// C is indexed by global vertex id; rows by (v - v0).
constexpr int kColoredCtr = 16;  // ctr slot counting `colored` pairs
struct SweepArgs {
    const int64_t *ro;
    const uint32_t *ci;
    uint32_t *C;
    const uint32_t *Fin;
    uint32_t *Fout;
    uint32_t *hub;
    unsigned long long *ctr;
    int64_t *nk;
    int64_t nk_cap;
    uint32_t k;
    int H;
    Keys keys;
    int dense;
    int64_t n_loc;
    uint32_t v0;
    uint32_t thread_max, hub_min;
    uint2 *colored;  // optional: (v, colour) of the vertices coloured this round
};
int sweep_round(const SweepArgs &a, cudaStream_t st, int blocks_sweep, int blocks_hub);

int ensure_scratch(gc_graph *g, bool need_event, bool need_luby);
int run_sweep_maxmin(gc_graph *g, const RunParams &p, RunResult *r);
int run_event_maxmin(gc_graph *g, const RunParams &p, RunResult *r);
int run_persistent_maxmin(gc_graph *g, const RunParams &p, RunResult *r);
int run_count_maxmin(gc_graph *g, const RunParams &p, RunResult *r);
int dedup_csr(gc_graph *g);  // gc_dedup.cu
int ensure_strict_rows(gc_graph *g);  // gc_dedup.cu: dedup first if a row is not strictly increasing
int run_count_jp(gc_graph *g, const RunParams &p, RunResult *r, int jpv);  // 1 Luby, 2 Alg.2, 3 Alg.4
int run_luby(gc_graph *g, const RunParams &p, RunResult *r);
int run_hash_is(gc_graph *g, const RunParams &p, int T, RunResult *r);  // gc_hash.cu (Alg.6)
int64_t count_colors_device(gc_graph *g, const uint32_t *C, int64_t n, bool compact,
                            uint32_t *C_inout, int64_t *launches, int64_t max_hint = -1);
int launch_priorities(uint64_t seed, int j, int64_t v_begin, int64_t count, uint32_t *out,
                      cudaStream_t st);

}  // namespace gc
