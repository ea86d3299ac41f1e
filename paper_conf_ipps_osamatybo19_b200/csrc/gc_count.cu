// gc_count.cu -- COUNT mode: the max-min colouring (Alg.1 + Alg.5, P:L102-113,
// P:L506-556; H = 1) computed from per-vertex COUNTS of uncoloured larger and
// smaller neighbours, all rounds in one persistent cooperative kernel with ONE
// grid barrier per round.
//
// Alg.5 L21-42 make v a local max in round k iff no neighbour u with
// R[u] > R[v] is still uncoloured at the start of round k (the snapshot of
// L26, R6), and a local min iff no smaller one is; v takes 2k+1 if min
// (min wins, R9), else 2k if max.  So with
//   hi(v) = #{u in adj(v) uncoloured, p(u) > p(v)},  lo(v) = same with <
// v is coloured in the first round k at whose start hi(v) == 0 or lo(v) == 0.
// Every vertex coloured in round k decrements, for each neighbour w, hi(w)
// (if it is larger than w) or lo(w) (if smaller), both halves of ONE 64-bit
// word, so the atomic returns both counts: the decrement that takes a side to
// zero while the other side is still positive is the unique first freeing of
// w -- it schedules w for round k+1 (w is min-coloured there if the freed side
// is lo).  If the other side is already zero, w was scheduled earlier; a lo
// side freed second stamps Zlo[w] = k+1, so a w scheduled by its hi side in
// round k still takes the min colour when lo was freed in the same round
// (min wins, Alg.5 L37-42, R9), and a stamp of round k+1 (k+2) never changes a
// decision of round k+1: the result is the snapshot result (Alg.5 L26, R6)
// for any interleaving.  Work: the row of every vertex is walked exactly once
// (when it is coloured) plus one counting pass, so a colouring is O(n + m);
// the walk issues no atomic for the neighbours on the side of v that was free
// (all coloured before v's round: their counts are dead), so fewer than one
// 8-byte atomic per directed entry; no witness search, no rescans.
//
// Kernels: the counting pass (k_count_zero + k_count_warp: 512-entry warp
// tiles over the column ids; k_count + k_count_hub for LDF / multi-hash)
// computes hi/lo of every vertex; k_count_persistent then colours round 0 in
// a dense init phase and runs rounds k = 0, 1, ... over the scheduled lists:
//   SL: rows of <= kShortMax entries, one 8-lane group each (4 entries/lane);
//   WL: longer rows as items of <= kSeg entries, one warp each.
// Work units (WL items, groups of 4 SL items) are dealt round-robin over the
// blocks, so every SM gets an equal share of a round's few thousand units.
// Items of round k are the slice [end_{k-1}, end_k) of two monotone arrays
// (each vertex is scheduled once, so the arrays never wrap).  At a round's
// end each block takes its slots among the next round's items for the
// vertices it freed, reserves them with its barrier arrival (one atomic on
// the round word) and writes them straight to their slots (fresh_flush_direct;
// the items carry round tags the consumers check).  Max-min rounds k >= 1 are
// relaxed (no release / acquire): the colours they write are provisional and
// one pass after the rounds applies the lo-freed-second stamps (DESIGN 7.0).

#include <cstdio>
#include <cstdlib>
#include <algorithm>

#include "gc_internal.cuh"

#ifndef GC_SKIP_COLOURED
#define GC_SKIP_COLOURED 0  // 1: walks test a status bit and skip coloured neighbours' atomics
                            // (measured on R-MAT s24: 38.7 vs 34.9 ms -- the extra dependent
                            // load costs more than the atomics it saves)
#endif

#ifndef GC_PREFETCH_WL
#define GC_PREFETCH_WL 0  // 1: prefetch the column ids of next round's long-row segments into L2
                          // (measured on R-MAT s24: 37.0 vs 35.0 ms -- the rounds are bound by
                          // the memory system's random traffic, extra requests slow them)
#endif

#ifndef GC_COUNT_STREAM
#define GC_COUNT_STREAM 1  // 1: counting pass of max-min / JP with random priorities as a tiled HBM
                           // stream (k_count_tile, double-buffered cp.async); 0: the degree-binned
                           // k_count + k_count_hub (always used for LDF and multi-hash)
#endif
constexpr bool kCountStream = GC_COUNT_STREAM != 0;

#ifndef GC_PROF_UNIT
#define GC_PROF_UNIT 0  // 1 (PROF builds only): per-round latency breakdown of the WL units
                        // (item load, column ids, atomics) in round_stats slots 9, 11-15
#endif

#ifndef GC_PROF_FRESH
#define GC_PROF_FRESH 0  // 1 (PROF builds only): end-of-round breakdown (fresh row loads, long-row
                         // expansion, flush reservation) in round_stats slots 9, 12, 14, 15
#endif

#ifndef GC_EAGER_RO
#define GC_EAGER_RO 0  // 1: the lane that frees w loads w's row offsets right away (max-min walk)
                       // instead of one thread per fresh vertex after the block's units
#endif

#ifndef GC_MERGED_HANDOFF
#define GC_MERGED_HANDOFF 1  // 1: a block's item reservation IS its barrier arrival (one release
                             // atomic), the staged items are copied while the barrier completes and
                             // carry round tags the consumers check; 0: reserve, copy, then arrive
#endif

#ifndef GC_SKIP_DEAD
#define GC_SKIP_DEAD 1  // 1: max-min walks skip the neighbours on the vertex's scheduling side
                        // (all coloured before its round: their counts are dead), see walk()
#endif
constexpr bool kSkipDead = GC_SKIP_DEAD != 0;

#ifndef GC_RELAXED_ARRIVE
#define GC_RELAXED_ARRIVE 1  // 1: max-min / multi-hash rounds k >= 1 arrive with a relaxed atomic and
                             // leave the barrier without an acquire fence (see stage_flush)
#endif
constexpr bool kRelaxedArrive = GC_RELAXED_ARRIVE != 0;


#ifndef GC_NO_PF_CI
#define GC_NO_PF_CI 1  // 1: no L2 prefetch of the next round's short rows (measured: 18.33 vs 18.43 ms with it)
#endif
#ifndef GC_NO_PF_RO
#define GC_NO_PF_RO 0  // experiments: no L2 prefetch of a freed vertex's row offsets
#endif

#ifndef GC_EAGER_FRESH
#define GC_EAGER_FRESH 0  // 1: max-min walks schedule the vertices they free right away (warp-level);
                          // measured 20.83 vs 18.10 ms on R-MAT s24: loads issued behind the round's atomics wait
#endif
constexpr bool kEagerFresh = GC_EAGER_FRESH != 0;

#ifndef GC_DIRECT_FLUSH
#define GC_DIRECT_FLUSH 1  // 1: max-min rounds reserve the next round's items right after the fresh
                           // vertices' row offsets are in, then write them straight to the lists
#endif
constexpr bool kDirectFlush = GC_DIRECT_FLUSH != 0;

#ifndef GC_INIT_TWO_PASS
#define GC_INIT_TWO_PASS 1  // 1: max-min init counts, reserves once per block, then writes round 0's items
#endif
constexpr bool kInitTwoPass = GC_INIT_TWO_PASS != 0;

#ifndef GC_PACKED
#define GC_PACKED 0  // 1: 32-bit (hi << 16 | lo) round counts -- max-min only (no JP / multi-hash branch);
                     // measured 27.9 vs 28.1 ms on R-MAT s24, not worth the restriction
#endif

namespace gc {

int ensure_nk(gc_graph *g, int64_t need);

namespace {

constexpr unsigned kFull = 0xFFFFFFFFu;
constexpr uint32_t kNone = 0xFFFFFFFFu;
constexpr uint32_t kNever = 0xFFFFFFFFu;  // Z: side never free (yet)
#ifndef GC_COUNT_THREADS
#define GC_COUNT_THREADS 512
#endif
#ifndef GC_COUNT_THREADS_MAXMIN
#define GC_COUNT_THREADS_MAXMIN 768  // measured on R-MAT s24 (max-min, relaxed rounds): 512 -> 18.9 ms,
                                     // 768 -> 18.4, 896 -> 19.2, 1024 -> 19.3 (64 registers)
#endif
constexpr int kThreads = GC_COUNT_THREADS;  // one block per SM (JP, multi-hash: more registers)
// threads per block of a kernel variant (max-min: 80 registers, no spills)
template <bool JP, bool MH>
constexpr int threads_for() { return (!JP && !MH) ? GC_COUNT_THREADS_MAXMIN : GC_COUNT_THREADS; }
constexpr int kThreadsMax = GC_COUNT_THREADS_MAXMIN > GC_COUNT_THREADS ? GC_COUNT_THREADS_MAXMIN : GC_COUNT_THREADS;
#ifndef GC_SHORT_MAX
#define GC_SHORT_MAX 32
#endif
#ifndef GC_SEG
#define GC_SEG 128  // measured on R-MAT s24: 128 -> 23.76 ms, 256 -> 23.90, 512 -> 28.4 (GC_SHORT_MAX 16: 24.1)
#endif
constexpr int kShortMax = GC_SHORT_MAX;    // SL rows: one 8-lane group
constexpr int kSeg = GC_SEG;               // WL item: one warp, kSeg / 32 entries per lane
constexpr int kHubMin = 4096;              // k_count: longer rows by blocks
constexpr uint32_t kInlineSeg = 4;         // schedule_fresh: rows of <= 4 segments written inline
constexpr int kHubChunk = 4096;
constexpr uint32_t kFirst = 0x80000000u;   // item flag: colour v in this round
constexpr uint32_t kLoSide = 0x40000000u;  // item flag: scheduled by its lo side (min colour)
constexpr uint32_t kLenMask = GC_MERGED_HANDOFF ? 0x3FFu : 0x3FFFFFFFu;  // merged: bits 10-29 hold the round tag
constexpr unsigned long long kDecHi = 0ull - (1ull << 32);
// Packed counts: the rounds decrement a 32-bit word (hi << 16 | lo) per vertex
// -- half the footprint of 64-bit words, so the round's burst of random
// atomics mostly hits L2 (tools/microbench_atomics.cu: a 205k-atomic burst
// takes 1.6 us on a 67 MB array, 3.6 us on 134 MB, whatever the width).
// Vertices of degree > kPackMax ("big") keep 64-bit words; they are few and
// are found through a hash set in shared memory (no extra global access).
constexpr int64_t kPackMax = 65535;
constexpr int kHTab = 4096;                // shared hash slots (big vertices <= kHTab / 2)
constexpr uint32_t kDec32Hi = 0u - (1u << 16);
constexpr unsigned long long kDecLo = ~0ull;

__device__ __forceinline__ unsigned lane_id() { return threadIdx.x & 31u; }

struct __align__(16) Item {
    uint32_t v;
    uint32_t lf;  // entry count | kFirst | kLoSide
    int64_t e0;   // first entry
};

// counters (each on its own 128-byte line where it is contended).  The item
// counts of round k's lists live in slot k % 3: round k reads slot k % 3,
// appends to slot (k+1) % 3 and clears slot (k+2) % 3 -- the last reader of
// that slot was round k-1's top, which every block has passed (a reader and
// a writer of one slot are always separated by a grid barrier).
enum : int {
    cS = 0,         // [0, 16, 32]: the round words R (SL items | WL items | barrier arrivals)
    cW = 48,        // [48, 64, 80]: (unused)
    cK = 96,        // [96, 112, 128]: vertices coloured in the round (stats)
    cCol = 144,     // vertices coloured (written at the end, host check)
    cBar = 160,     // (unused: arrivals live in the round words)
    cFin = 168,     // relaxed rounds: the final release / acquire barrier
    cMaxC = 171,    // relaxed rounds: 1 + the largest colour (0: none)
    cAbort = 176,
    cErr = 192,     // [192..194] first trap: kind, round, vertex
    cRounds = 208,  // result: rounds R
    cIters = 209,   // loop iterations run
    cVis = 210,     // PROF: entries walked in the rounds
    cPhaseNs = 211, // PROF: ns in the init phase, the rounds
    cHubs = 224,    // k_count: hub rows
    cSlot = 240,    // JP: mex slots handed out (monotone)
    cRW = 256,      // round words: [16 * (slot * kNG + group)], 3 rotating slots x kNG groups
    kCCtrWords = 512
};

struct CArgs {
    const int64_t *ro;
    const uint32_t *ci;
    uint32_t *C;
    unsigned long long *cnt;  // (hi << 32) | lo from the counting kernels (read by init)
    uint32_t *cnt32;          // the rounds' counts: (hi << 16) | lo per vertex, or ...
    uint32_t *big32;          // ... for big vertices, [2 s] = hi, [2 s + 1] = lo, [2 kHTab + s] =
                              // "scheduled" flag, s = the vertex's slot in the shared hash set
    const uint32_t *big;      // big vertices (degree > kPackMax)
    int nbig;
    uint32_t *Zlo;            // round from which lo is free, when freed second (else kNever)
    Item *SL;
    Item *WL;
    unsigned long long *ctr;
    int64_t *nk;
    int64_t *rstat;
    int64_t nk_cap;
    int64_t n;
    uint32_t key;
    uint32_t max_rounds;
    unsigned long long sl_cap, wl_cap;
    uint32_t *jslot;               // JP: mex slots of long rows (kSlotWords each)
    unsigned long long jslot_cap;
    uint32_t *M;                   // status bits: 1 = uncoloured (max-min, multi-hash)
    int jpv;                       // JP kernel: 1 Luby (mex), 2 Alg.2 max-only, 3 Alg.2 + Alg.4
    uint32_t *cr;                  // Alg.4: colour of each round
    uint32_t *B;                   // Alg.4: 3 colour sets of bwords words (round k: B + (k % 3) * bwords)
    uint32_t bwords;
    int H;                         // MH: weight functions (count words v * H + j)
    uint32_t mkeys[GC_MAX_HASHES]; // MH: their keys K_j
    const uint32_t *dg;            // LDF: vertex degrees; nullptr = weights only
    uint32_t epoch;                // colourings run on this handle (item round tags)
    int jrel;                      // JP Luby / Alg.2 rounds relaxed (jp_colour_of, jp_segment_done)
};

// Round tags of the items walked in round r (merged hand-off): items are
// written after their producer's barrier arrival, so a consumer checks that
// both 8-byte halves of an item carry round r's tag (each half is written by
// one 8-byte element store, single-copy atomic) and re-reads until they do.
// The epoch separates colourings (the arrays are cleared every 256).
__device__ __forceinline__ uint32_t tag_a(uint32_t epoch, uint32_t r) { return ((epoch & 0xFu) << 16) | (r & 0xFFFFu); }
__device__ __forceinline__ uint32_t tag_b(uint32_t epoch, uint32_t r) { return ((epoch & 0xFFu) << 16) | (r & 0xFFFFu); }

// Priority key of v (R1; with LDF the (degree, weight) pair of R21 as one
// 64-bit integer, degree in the high half): comparisons of keys are the
// comparisons of Alg.5 L29-34 / Alg.2 L9.
__device__ __forceinline__ uint64_t prio_key(const CArgs &a, uint32_t v) {
    const uint64_t w = weight_mix(v ^ a.key);
    return (a.dg && v != 0xFFFFFFFFu) ? w | ((uint64_t)__ldg(a.dg + v) << 32) : w;  // (kNone: a hole item)
}
// JP mex slot of a long row: a 1024-bit presence set of its predecessors'
// colours + the number of its entries not yet walked (the segment that takes
// it to zero computes the mex and writes the colour).
constexpr int kSlotWords = 36;  // [0, 32) bits, [32] entries remaining
constexpr uint32_t kMexWin = 1024;

__device__ __forceinline__ void flag_error(const CArgs &a, unsigned kind, uint32_t k, uint32_t v) {
    if (atomicCAS(&a.ctr[cErr], 0ull, (unsigned long long)kind) == 0ull) {
        a.ctr[cErr + 1] = k;
        a.ctr[cErr + 2] = v;
    }
}

__device__ __forceinline__ unsigned long long gtimer() {
    unsigned long long t;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
    return t;
}
__device__ __forceinline__ unsigned long long ld_acquire(const unsigned long long *p) {
    unsigned long long v;
    asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ unsigned long long atom_add_release(unsigned long long *p,
                                                               unsigned long long x) {
    unsigned long long v;
    asm volatile("atom.add.release.gpu.global.u64 %0, [%1], %2;" : "=l"(v) : "l"(p), "l"(x) : "memory");
    return v;
}

// 64-bit add on GLOBAL memory.  atomicAdd through a generic pointer (CArgs
// members) compiles to ATOM.E + a shared-memory CAS fallback branch, which
// serialises a lane's atomics (each waits for the previous one's predicate);
// the global form lets all Q atomics of a lane be in flight together.
__device__ __forceinline__ unsigned long long atom_add_global(unsigned long long *p,
                                                              unsigned long long x) {
    unsigned long long old;
    asm volatile("atom.global.add.u64 %0, [%1], %2;" : "=l"(old) : "l"(p), "l"(x));
    return old;
}

// fire-and-forget PROF counters (no wait for a result)
__device__ __forceinline__ void red_max(int64_t *p, unsigned long long x) {
    asm volatile("red.global.max.u64 [%0], %1;" ::"l"(p), "l"(x) : "memory");
}
__device__ __forceinline__ void red_add(int64_t *p, unsigned long long x) {
    asm volatile("red.global.add.u64 [%0], %1;" ::"l"(p), "l"(x) : "memory");
}
__device__ __forceinline__ uint32_t atom_or_global(uint32_t *p, uint32_t x) {
    uint32_t old;
    asm volatile("atom.global.or.b32 %0, [%1], %2;" : "=r"(old) : "l"(p), "r"(x));
    return old;
}
__device__ __forceinline__ uint32_t atom_add_global32(uint32_t *p, uint32_t x) {
    uint32_t old;
    asm volatile("atom.global.add.u32 %0, [%1], %2;" : "=r"(old) : "l"(p), "r"(x));
    return old;
}

// Round words (3 rotating slots per group): SL item count in bits [0, 29),
// WL item count in [29, 53), barrier arrivals in [53, 64).  The blocks are
// split into kNG groups (block b: group b % kNG), each with its own round
// words and item arrays, so a word takes ~G / kNG same-address atomics per
// round instead of G (they serialise in one L2 slice).  A block reserves its
// items of the next round with ONE atomic on its group's word (both list
// bases come back); the spin that ends the round's barrier loads every
// group's word and so reads the next round's item counts in the same loads
// that see the last arrivals.
#ifndef GC_BARRIER_GROUPS
#define GC_BARRIER_GROUPS 1  // measured on R-MAT s24 (persistent kernel): 1 group 23.9 ms, 2: 24.5, 4: 26.0, 8: 29.7
#endif
constexpr int kNG = GC_BARRIER_GROUPS;
#ifndef GC_BARRIER_RELAXED_SPIN
#define GC_BARRIER_RELAXED_SPIN 1
#endif
__device__ __forceinline__ unsigned long long ld_relaxed_u64(const unsigned long long *p) {
    unsigned long long v;
    asm volatile("ld.relaxed.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}
constexpr unsigned long long kRwWL = 1ull << 29, kRwArr = 1ull << 53;
constexpr unsigned long long kMSL = kRwWL - 1ull, kMWL = (1ull << 24) - 1ull;
__device__ __forceinline__ unsigned long long rw_field(unsigned long long v, int li) {
    return li == 0 ? (v & kMSL) : ((v >> 29) & kMWL);
}
__device__ __forceinline__ unsigned long long rw_add(unsigned long long c, int li) {
    return li == 0 ? c : c << 29;
}

// Grid barrier over the round words of ring slot `slot` (all blocks resident,
// cooperative launch): release arrival on the block's group word, acquire
// spin over all groups' words (which also invalidates the SM's L1, so the
// next phase sees what other SMs wrote); thread 0 leaves the final words in
// out[0..kNG).  A wait beyond 4 s records a trap and makes every block leave
// instead of hanging the GPU.
__device__ __forceinline__ unsigned long long *round_word(const CArgs &a, int slot, int grp) {
    return a.ctr + cRW + 16 * (slot * kNG + grp);
}
__device__ __forceinline__ unsigned group_size(int grp) {
    return (gridDim.x - (unsigned)grp + kNG - 1) / kNG;
}
__device__ __forceinline__ bool grid_barrier_rw(const CArgs &a, uint32_t k, int slot,
                                                unsigned long long *out, bool acquire = true) {
    __shared__ int ok_sh;
    __syncthreads();
    if (threadIdx.x == 0) {
        int ok = 1;
#if GC_MERGED_HANDOFF
        // (the block arrived with its item reservation in stage_flush)
#elif GC_BARRIER_RELAXED_SPIN
        // arrival without a return value (release pattern), relaxed spin,
        // one acquire fence after the last arrival is seen
        asm volatile("red.release.gpu.global.add.u64 [%0], %1;" ::"l"(round_word(a, slot, (int)(blockIdx.x % kNG))),
                     "l"(kRwArr) : "memory");
#else
        atom_add_release(round_word(a, slot, (int)(blockIdx.x % kNG)), kRwArr);
#endif
        unsigned spins = 0;
        const unsigned long long t0 = gtimer();
        for (;;) {
            bool done = true;
#pragma unroll
            for (int gq = 0; gq < kNG; ++gq) {
#if GC_BARRIER_RELAXED_SPIN
                out[gq] = ld_relaxed_u64(round_word(a, slot, gq));
#else
                out[gq] = ld_acquire(round_word(a, slot, gq));
#endif
                done = done && (out[gq] >> 53) >= group_size(gq);
            }
            if (done) {
#if GC_BARRIER_RELAXED_SPIN
                if (acquire) asm volatile("fence.acq_rel.gpu;" ::: "memory");
#endif
                break;
            }
            if ((++spins & 255u) == 0u) {
                if (*(volatile unsigned long long *)(a.ctr + cAbort)) {
                    ok = 0;
                    break;
                }
                if (gtimer() - t0 > 4000000000ull) {
                    flag_error(a, 100, k, blockIdx.x);
                    atomicExch(a.ctr + cAbort, 1ull);
                    ok = 0;
                    break;
                }
            }
        }
        ok_sh = ok;
    }
    __syncthreads();
    return ok_sh != 0;
}


// ---------------------------------------------------------------- staging
// Staging sizes: a typical round has ~25 items per block (round 0 spills to
// the global lists anyway).  The Stage size sets the shared-memory carveout
// and so the L1 left to the kernel.  While the kernel kept a local copy of
// its parameters (before __grid_constant__, below) L1 decided a lot (R-MAT
// s24: 198 KB of Stage, 28 KB L1: 39.0 ms; 194 KB: 34.2; 20 KB: 31.1); with
// the parameters read in place: 1024 items 28.6 ms, 256 items 28.7 ms.
#ifndef GC_STAGE_ITEMS
#define GC_STAGE_ITEMS 1024
#endif
constexpr int kStS = GC_STAGE_ITEMS, kStW = GC_STAGE_ITEMS, kStF = 2 * GC_STAGE_ITEMS,
              kLongMax = GC_STAGE_ITEMS / 4;
constexpr int kCSetWords = 1024;  // Alg.4: colours < 32768 collected in shared memory
struct Stage {
    Item s[kStS];
    Item w[kStW];
    uint2 fresh[kStF];              // (w, lo side?) this block scheduled in the round
    int64_t frs[kStF];              // direct flush: their row starts ...
    uint2 fmeta[kStF];              // ... (row length, first slot among the block's direct items)
    unsigned nd[2];                 // direct flush: the block's direct SL items / WL segments
#if GC_EAGER_RO
    longlong2 fro[kStF];            // their row offsets (loaded by the freeing lane)
#endif
#if GC_PACKED
    uint32_t htab[kHTab];           // hash set of the big vertices (kNone = empty)
#endif
    uint32_t wbits[kThreadsMax / 32][32];  // JP: per-warp 1024-bit mex window
    uint32_t cset[kCSetWords];          // Alg.4: the block's share of the round's colour set
    uint32_t cprev;                     // Alg.4: colour of the previous round
    unsigned cmin;                      // Alg.4: block reduction scratch
    struct Long {                   // schedule_fresh: a long row to expand
        int64_t rs, dst;            // row start; first item slot (>= 0 staged, < 0: ~global)
        uint32_t w, len, flags, pad;
    } lng[kLongMax];
    unsigned nlong;
    unsigned nf;
    unsigned n[2];
    unsigned colored;
    unsigned vis;                   // PROF: entries walked by this block in the round
    unsigned long long t_fs;        // PROF: when this block's fresh step started
    unsigned long long base[2];
    // append targets of the current round (set by thread 0 at the round top)
    unsigned long long *rw;         // the next round's word R (item reservations, arrivals)
    unsigned long long nbase[2];    // where the next round's items start
    unsigned long long *ccol;       // coloured-count slot of this round
    uint32_t tg_a, tg_b;            // round tags of the items appended now (next round's)
    unsigned long long rd[kNG];     // the groups' round words from the barrier
    unsigned long long gn[2][kNG + 1];  // per list: prefix of the groups' item counts of the round
    unsigned long long g0[2][kNG];  // per list and group: where the round's items start
    unsigned long long trap;
};
constexpr size_t kStageBytes = sizeof(Stage);

__device__ __forceinline__ Stage &stage() {
    extern __shared__ __align__(16) unsigned char smem_raw[];
    return *reinterpret_cast<Stage *>(smem_raw);
}

__device__ __forceinline__ unsigned hslot(uint32_t v) { return (v * 2654435761u) >> 20; }  // 12 bits
// slot of v in the block's hash set of big vertices, or -1
__device__ __forceinline__ int big_slot(uint32_t v) {
#if GC_PACKED
    const uint32_t *t = stage().htab;
    for (unsigned h = hslot(v);; h = (h + 1) & (kHTab - 1)) {
        const uint32_t x = t[h];
        if (x == v) return (int)h;
        if (x == kNone) return -1;
    }
#else
    (void)v;
    return -1;
#endif
}

// this block's group's item array of list li (offset into SL / WL)
__device__ __forceinline__ size_t grp_base(const CArgs &a, int li) {
    return (size_t)(blockIdx.x % kNG) * (size_t)(li == 0 ? a.sl_cap : a.wl_cap);
}
// the group and index (into that group's array) of item t of the round's
// list li (items numbered group by group)
__device__ __forceinline__ const Item *round_item(const CArgs &a, int li, unsigned long long t) {
    const Stage &st = stage();
    int gq = 0;
#pragma unroll
    for (int x = 1; x < kNG; ++x) gq += t >= st.gn[li][x] ? 1 : 0;
    return (li == 0 ? a.SL + (size_t)gq * a.sl_cap : a.WL + (size_t)gq * a.wl_cap) + st.g0[li][gq] +
           (t - st.gn[li][gq]);
}

// an item of the next round into global memory (tagged under the merged hand-off)
__device__ __forceinline__ void gput(Item *p, const Item &v) {
#if GC_MERGED_HANDOFF
    const Stage &st = stage();
    // (a hole's lf / e0 may be uninitialised shared memory: masked to their fields)
    const unsigned long long w0 =
        (unsigned long long)v.v | ((unsigned long long)((v.lf & 0xC00003FFu) | (st.tg_a << 10)) << 32);
    const unsigned long long w1 = ((unsigned long long)v.e0 & ((1ull << 40) - 1ull)) | ((unsigned long long)st.tg_b << 40);
    asm volatile("st.relaxed.gpu.global.v2.u64 [%0], {%1, %2};" ::"l"(p), "l"(w0), "l"(w1) : "memory");
#else
    *p = v;
#endif
}
// an item of round k (merged hand-off: until both halves carry its tags)
__device__ __forceinline__ Item gget(const CArgs &a, const Item *p, uint32_t k) {
    Item it;
#if GC_MERGED_HANDOFF
    const uint32_t ta = tag_a(a.epoch, k), tb = tag_b(a.epoch, k);
    unsigned long long w0, w1;
    for (unsigned spins = 0;; ++spins) {
        asm volatile("ld.relaxed.gpu.global.v2.u64 {%0, %1}, [%2];" : "=l"(w0), "=l"(w1) : "l"(p) : "memory");
        if ((((uint32_t)(w0 >> 32) >> 10) & 0xFFFFFu) == ta && (uint32_t)(w1 >> 40) == tb) break;
        if (spins > (1u << 24)) {  // ~seconds: an item that never arrives (cannot happen)
            flag_error(a, 11, k, (uint32_t)w0);
            break;
        }
    }
    it.v = (uint32_t)w0;
    it.lf = (uint32_t)(w0 >> 32) & ~(0xFFFFFu << 10);
    it.e0 = (int64_t)(w1 & ((1ull << 40) - 1ull));
#else
    (void)a;
    (void)k;
    it = *p;
#endif
    return it;
}

// Whole warp converged: lanes with `pred` append `val` to staged list li;
// beyond the shared capacity the entries go straight to the global list.
__device__ __forceinline__ void stage_append(const CArgs &a, bool pred, const Item &val, int li) {
    const unsigned m = __ballot_sync(kFull, pred);
    if (!m) return;
    Stage &st = stage();
    const unsigned lane = lane_id();
    const unsigned leader = __ffs(m) - 1;
    unsigned base = 0;
    if (lane == leader) base = atomicAdd(&st.n[li], (unsigned)__popc(m));
    base = __shfl_sync(kFull, base, leader);
    const unsigned pos = base + __popc(m & ((1u << lane) - 1u));
    const unsigned cap = li == 0 ? kStS : kStW;
    Item *buf = li == 0 ? st.s : st.w;
    const bool spill = pred && pos >= cap;
    if (pred && !spill) buf[pos] = val;
    const unsigned sm = __ballot_sync(kFull, spill);
    if (sm) {
        const unsigned sl = __ffs(sm) - 1;
        unsigned long long gb = 0;
        if (lane == sl) gb = rw_field(atom_add_global(st.rw, rw_add((unsigned long long)__popc(sm), li)), li);
        gb = __shfl_sync(kFull, gb, sl);
        if (spill) {
            const unsigned long long at = st.nbase[li] + gb + __popc(sm & ((1u << lane) - 1u));
            const unsigned long long capg = li == 0 ? a.sl_cap : a.wl_cap;
            if (at < capg) gput((li == 0 ? a.SL + grp_base(a, 0) : a.WL + grp_base(a, 1)) + at, val);
            else flag_error(a, 1, 0, val.v);
        }
    }
}

// Whole block: move staged items to the global lists, add the coloured count.
// PROF: prs = this round's stat record (entries walked, longest block work).
// relaxed (max-min rounds k >= 1): the arrival needs no release because no
// later round reads anything the round writes through a plain load: items
// carry round tags and are re-read until both halves do, the counts are
// atomics, and the lo-freed-second stamps and the colours are read only after
// the rounds, behind one release / acquire barrier (the final pass of
// k_count_persistent).
__device__ __forceinline__ void stage_flush(const CArgs &a, int64_t *prs = nullptr,
                                            unsigned long long t_round = 0, bool relaxed = false) {
    Stage &st = stage();
    __syncthreads();
    if (prs && threadIdx.x == 0) {
        const unsigned long long fdt = gtimer() - st.t_fs;  // this block's fresh step
        if (!GC_PROF_UNIT) {
            red_add(prs + 11, fdt);
            red_max(prs + 12, fdt);
        }
        red_add(prs + 2, (unsigned long long)st.vis);
        red_max(prs + 5, gtimer() - t_round);
        st.vis = 0;
    }
    if (threadIdx.x == 0) {
        // both reservations in flight together (each is an L2 round trip)
        const unsigned c0 = min(st.n[0], (unsigned)kStS), c1 = min(st.n[1], (unsigned)kStW);
        // the round's coloured count (statistics: the frontier trace; under
        // relaxed arrivals the completion check counts the colours instead)
        if (st.colored) atom_add_global(st.ccol, (unsigned long long)st.colored);
        st.colored = 0;
#if GC_MERGED_HANDOFF
        // one reservation for both lists, which is also the barrier arrival:
        // the release orders every earlier write of the block (colours, Z
        // stamps, spilled items); the staged items follow, tagged
        const unsigned long long rv = relaxed ? atom_add_global(st.rw, rw_add(c0, 0) + rw_add(c1, 1) + kRwArr)
                                              : atom_add_release(st.rw, rw_add(c0, 0) + rw_add(c1, 1) + kRwArr);
#else
        // one reservation for both lists
        const unsigned long long rv = (c0 || c1) ? atom_add_global(st.rw, rw_add(c0, 0) + rw_add(c1, 1)) : 0ull;
#endif
        if (GC_PROF_FRESH && prs) {  // the reservation came back
            asm volatile("" ::"l"(rv));
            red_max(prs + 9, gtimer() - t_round);
        }
        const unsigned long long r0 = rw_field(rv, 0), r1 = rw_field(rv, 1);
        if (r0 + c0 > kMSL || r1 + c1 > kMWL) flag_error(a, 9, 0, 0);  // a round word field overflowed
        st.n[0] = c0;
        st.n[1] = c1;
        st.base[0] = c0 ? st.nbase[0] + r0 : 0ull;
        st.base[1] = c1 ? st.nbase[1] + r1 : 0ull;
        for (int i = 0; i < 2; ++i) {
            const unsigned long long capg = i == 0 ? a.sl_cap : a.wl_cap;
            if (st.n[i] && st.base[i] + st.n[i] > capg) {
                flag_error(a, 2, 0, (unsigned)i);
                st.n[i] = 0;
            }
        }
        st.nf = 0;
    }
    __syncthreads();
    Item *const sl = a.SL + grp_base(a, 0), *const wl = a.WL + grp_base(a, 1);
    for (unsigned i = threadIdx.x; i < st.n[0]; i += blockDim.x) gput(sl + st.base[0] + i, st.s[i]);
    for (unsigned i = threadIdx.x; i < st.n[1]; i += blockDim.x) gput(wl + st.base[1] + i, st.w[i]);
    __syncthreads();
    if (threadIdx.x < 2) st.n[threadIdx.x] = 0;
    if (prs && threadIdx.x == 0)
        red_max(prs + 8, gtimer() - t_round);
}

// Whole block, end of a max-min round (relaxed rounds, kDirectFlush): one
// thread per fresh vertex loads its row offsets and takes its slots among
// the block's items of the next round (an SL item, or its WL segments); the
// block then reserves them with its arrival (one relaxed atomic on the round
// word) and writes every item straight to its slot -- long rows expanded by
// a warp each -- while the barrier completes (the items carry round tags the
// consumers check).  Items staged in shared memory by the rare overflow
// paths of the walks go first.
__device__ __forceinline__ void jp_slot_init(const CArgs &a, uint32_t w, int64_t deg);  // (below)

template <bool JP>
__device__ __forceinline__ void fresh_flush_direct(const CArgs &a, bool relaxed, int64_t *prs = nullptr,
                                                   unsigned long long t_round = 0) {
    Stage &st = stage();
    __syncthreads();  // the units are done
    if (prs && threadIdx.x == 0) {  // PROF (round_stats slots as the staged flush's, tools/freshprof.py)
        red_max(prs + 7, gtimer() - t_round);
        red_add(prs + 2, (unsigned long long)st.vis);
        st.vis = 0;
    }
    const unsigned nf = min(st.nf, (unsigned)kStF);
    for (unsigned t = threadIdx.x; t < nf; t += blockDim.x) {
        const uint2 f = st.fresh[t];
        const int64_t rs = a.ro[f.x], re = a.ro[f.x + 1];
        const int64_t len = re - rs;
        unsigned pos;
        if (len <= kShortMax) {
            pos = atomicAdd(&st.nd[0], 1u);
            if (!GC_NO_PF_CI && len > 0) asm volatile("prefetch.global.L2 [%0];" ::"l"(a.ci + rs));
        } else {
            pos = atomicAdd(&st.nd[1], (unsigned)((len + kSeg - 1) / kSeg));
            if (JP && a.jpv == 1) jp_slot_init(a, f.x, len);  // (before the release arrival)
        }
        st.frs[t] = rs;
        st.fmeta[t] = make_uint2((uint32_t)len, pos);
    }
    __syncthreads();
    if (prs && threadIdx.x == 0) {  // PROF: the fresh vertices' row offsets are in, slots taken
        red_max(prs + 14, gtimer() - t_round);
        red_max(prs + 5, gtimer() - t_round);
    }
    if (threadIdx.x == 0) {
        const unsigned c0 = min(st.n[0], (unsigned)kStS), c1 = min(st.n[1], (unsigned)kStW);
        const unsigned long long t0 = c0 + st.nd[0], t1 = c1 + st.nd[1];
        if (st.colored) atom_add_global(st.ccol, (unsigned long long)st.colored);
        st.colored = 0;
        // the reservation of both lists is the barrier arrival (relaxed for
        // max-min, 7.0; release for JP, whose mex reads earlier colours)
        const unsigned long long rv = relaxed ? atom_add_global(st.rw, rw_add(t0, 0) + rw_add(t1, 1) + kRwArr)
                                              : atom_add_release(st.rw, rw_add(t0, 0) + rw_add(t1, 1) + kRwArr);
        const unsigned long long r0 = rw_field(rv, 0), r1 = rw_field(rv, 1);
        if (prs) {  // PROF: the reservation (= arrival) came back
            asm volatile("" ::"l"(rv));
            red_max(prs + 9, gtimer() - t_round);
        }
        if (r0 + t0 > kMSL || r1 + t1 > kMWL) flag_error(a, 9, 0, 0);  // a round word field overflowed
        st.base[0] = st.nbase[0] + r0;
        st.base[1] = st.nbase[1] + r1;
        st.n[0] = c0;
        st.n[1] = c1;
        if (st.base[0] + t0 > a.sl_cap || st.base[1] + t1 > a.wl_cap) {
            flag_error(a, 2, 0, 0);
            st.n[0] = st.n[1] = 0;
            st.nf = 0;
        }
        st.nlong = 0;
    }
    __syncthreads();
    Item *const sl = a.SL + grp_base(a, 0), *const wl = a.WL + grp_base(a, 1);
    const unsigned c0 = st.n[0], c1 = st.n[1];
    const unsigned long long b0 = st.base[0], b1 = st.base[1];
    for (unsigned i = threadIdx.x; i < c0; i += blockDim.x) gput(sl + b0 + i, st.s[i]);
    for (unsigned i = threadIdx.x; i < c1; i += blockDim.x) gput(wl + b1 + i, st.w[i]);
    const unsigned nf2 = min(st.nf, (unsigned)kStF);
    for (unsigned t = threadIdx.x; t < nf2; t += blockDim.x) {
        const uint2 f = st.fresh[t];
        const uint2 mt = st.fmeta[t];
        const int64_t rs = st.frs[t], len = (int64_t)mt.x;
        const uint32_t fl = kFirst | f.y;
        if (len <= kShortMax) {
            Item it;
            it.v = f.x;
            it.lf = (uint32_t)len | fl;
            it.e0 = rs;
            gput(sl + b0 + c0 + mt.y, it);
        } else {
            const uint32_t nseg = (uint32_t)((len + kSeg - 1) / kSeg);
            const unsigned li = nseg <= kInlineSeg ? (unsigned)kLongMax : atomicAdd(&st.nlong, 1u);
            if (li < (unsigned)kLongMax) {
                st.lng[li].rs = rs;
                st.lng[li].dst = (int64_t)(c1 + mt.y);
                st.lng[li].w = f.x;
                st.lng[li].len = (uint32_t)len;
                st.lng[li].flags = fl;
            } else {
                for (uint32_t q = 0; q < nseg; ++q) {
                    Item si;
                    si.v = f.x;
                    si.e0 = rs + (int64_t)q * kSeg;
                    si.lf = (uint32_t)min((int64_t)kSeg, len - (int64_t)q * kSeg) |
                            ((q == 0 || (JP && a.jpv == 1)) ? fl : (fl & kLoSide));
                    gput(wl + b1 + c1 + mt.y + q, si);
                }
            }
        }
    }
    __syncthreads();
    if (prs && threadIdx.x == 0) red_max(prs + 15, gtimer() - t_round);  // PROF: short items written
    const unsigned nl = min(st.nlong, (unsigned)kLongMax);
    for (unsigned r = threadIdx.x >> 5; r < nl; r += blockDim.x >> 5) {  // a warp per long row
        const Stage::Long L = st.lng[r];
        const uint32_t nseg = (L.len + kSeg - 1) / kSeg;
        for (uint32_t q = lane_id(); q < nseg; q += 32) {
            Item si;
            si.v = L.w;
            si.e0 = L.rs + (int64_t)q * kSeg;
            si.lf = (uint32_t)min((int64_t)kSeg, (int64_t)L.len - (int64_t)q * kSeg) |
                    ((q == 0 || (JP && a.jpv == 1)) ? L.flags : (L.flags & kLoSide));
            gput(wl + b1 + L.dst + q, si);
        }
    }
    if (prs) {  // PROF: every item written
        __syncthreads();
        if (threadIdx.x == 0) red_max(prs + 8, gtimer() - t_round);
    }
    // (st.n, st.nd, st.nf are reset at the next round top)
}

// JP: a mex slot for the long row of w (deg entries): cleared, its
// remaining-entry count set, its index kept in Zlo[w] (JP has no lo side).
__device__ __forceinline__ void jp_slot_init(const CArgs &a, uint32_t w, int64_t deg) {
    const unsigned long long s = atom_add_global(a.ctr + cSlot, 1ull);
    if (s >= a.jslot_cap) {
        flag_error(a, 6, 0, w);
        return;
    }
    if (!a.jrel) {  // (relaxed rounds: the host zeroes every slot before the colouring)
        uint4 *p = reinterpret_cast<uint4 *>(a.jslot + s * kSlotWords);
#pragma unroll
        for (int i = 0; i < kSlotWords / 4; ++i) p[i] = make_uint4(0u, 0u, 0u, 0u);
        a.jslot[s * kSlotWords + 32] = (uint32_t)deg;
    }
    a.Zlo[w] = (uint32_t)s;
}

// JP, relaxed rounds: a value written once in an earlier round by another
// block (a predecessor's colour, a row's slot index) is read until it is no
// longer the initial one -- a single-writer word that changes once, so the
// value read then is the value written, whatever the ordering
__device__ __forceinline__ uint32_t jp_read_once(const CArgs &a, const uint32_t *p, uint32_t init, uint32_t k,
                                                 uint32_t v) {
    uint32_t x = __ldcg(p);
    for (unsigned spins = 0; x == init; ++spins) {
        if (spins > (1u << 22)) {  // (~ms: the writer's round is long over -- cannot happen)
            flag_error(a, 5, k, v);
            break;
        }
        x = __ldcg(p);
    }
    return x;
}

// Whole warp converged: schedule the rows of the lanes with `pred` (vertex w,
// row [rs, rs + len)) for the next round: short rows as one SL item, longer
// rows as ceil(len / kSeg) WL items (expanded by the whole warp).  JP: every
// segment of a row to be coloured carries the flags (each feeds the mex).
template <bool JP>
__device__ __forceinline__ void schedule_rows(const CArgs &a, bool pred, uint32_t w, int64_t rs,
                                              int64_t len, uint32_t ff) {
    const bool shortrow = pred && len <= kShortMax;
    Item it;
    it.v = w;
    it.lf = (uint32_t)len | ff;
    it.e0 = rs;
    if (shortrow && len > 0) {  // the row walked next round: HBM -> L2 now (<= 2 lines)
        if (!GC_NO_PF_CI) asm volatile("prefetch.global.L2 [%0];" ::"l"(a.ci + rs));
        if (!GC_NO_PF_CI) asm volatile("prefetch.global.L2 [%0];" ::"l"(a.ci + rs + len - 1));
    }
    stage_append(a, shortrow, it, 0);
    unsigned lm = __ballot_sync(kFull, pred && !shortrow);
    while (lm) {
        const int src = __ffs(lm) - 1;
        lm &= lm - 1;
        const uint32_t ww = __shfl_sync(kFull, w, src);
        const int64_t r0 = __shfl_sync(kFull, rs, src);
        const int64_t ln = __shfl_sync(kFull, len, src);
        const uint32_t fs = __shfl_sync(kFull, ff, src);
        if (JP && a.jpv == 1 && (fs & kFirst) && lane_id() == 0) jp_slot_init(a, ww, ln);
        const uint32_t nseg = (uint32_t)((ln + kSeg - 1) / kSeg);
        for (uint32_t q0 = 0; q0 < nseg; q0 += 32) {
            const uint32_t q = q0 + lane_id();
            Item si;
            si.v = ww;
            const int64_t e0 = r0 + (int64_t)q * kSeg;
            si.e0 = e0;
            si.lf = (uint32_t)min((int64_t)kSeg, r0 + ln - e0) | ((q == 0 || (JP && a.jpv == 1)) ? fs : (fs & kLoSide));
            stage_append(a, q < nseg, si, 1);
        }
    }
}

// Out-of-line copy for the rare paths inside the unrolled walk (overflowing
// fresh list): keeps walk's code and registers small.
template <bool JP>
__device__ __noinline__ void schedule_rows_slow(const CArgs &a, bool pred, uint32_t w, int64_t rs,
                                                int64_t len, uint32_t ff) {
    schedule_rows<JP>(a, pred, w, rs, len, ff);
}

// v leaves the uncoloured set: its status bit is cleared (later walks skip
// its count; a coloured vertex's counts no longer decide anything)
__device__ __forceinline__ void clear_status(const CArgs &a, uint32_t v) {
    if (GC_SKIP_COLOURED) atomicAnd(a.M + (v >> 5), ~(1u << (v & 31u)));
}


// Walk entries e, e + stride, ... (< end, Q of them) of the row of v coloured
// in round k (v == kNone: idle lane; whole warp converged): decrement the
// side of each neighbour w that v belongs to; a side reaching zero is free
// from round k+1 and schedules w (first time only).
// JP (the Luby-MIS variant as first-fit greedy in decreasing weight order,
// R10): only the hi side exists (lo is pinned at 1); the entries w LARGER than
// v are v's already-coloured predecessors -- their colours go into v's mex
// set: bits < 64 of `mask` (short rows), or bits < 1024 of the warp's shared
// bitmap `sbits` (WIDE: long-row segments).  mex = `want_mex` lanes only.
template <int Q, bool JP = false, bool WIDE = false>
__device__ __forceinline__ void walk(const CArgs &a, uint32_t v, uint64_t pv, int64_t e,
                                     int64_t end, int stride, uint32_t k, uint32_t &nvis,
                                     unsigned long long *mask = nullptr, uint32_t *sbits = nullptr,
                                     bool want_mex = false, bool want_set = false,
                                     long long *tprof = nullptr, int skipside = -1) {
    uint32_t w[Q];
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        const int64_t eq = e + (int64_t)q * stride;
        w[q] = (v != kNone && eq < end) ? __ldcs(a.ci + eq) : kNone;
    }
    if (GC_PROF_UNIT && tprof) {
#pragma unroll
        for (int q = 0; q < Q; ++q) asm volatile("" ::"r"(w[q]));
        tprof[0] = clock64();
    }
    if (!JP && GC_SKIP_COLOURED) {  // coloured neighbours: no atomic (their counts are dead)
        uint32_t mb[Q];
#pragma unroll
        for (int q = 0; q < Q; ++q) mb[q] = w[q] != kNone ? __ldcg(a.M + (w[q] >> 5)) : 0u;
#pragma unroll
        for (int q = 0; q < Q; ++q)
            if (w[q] != kNone && !((mb[q] >> (w[q] & 31u)) & 1u)) w[q] = kNone;
    }
    // One atomic per entry, address and value chosen without a branch
    // (a branch around each atomic made the compiler wait for every result).
#if GC_PACKED
    uint32_t old[Q];
#else
    unsigned long long old[Q];
#endif
    bool hi[Q];
    int slot[Q];
    uint32_t cv[Q];  // JP: colours of the larger neighbours
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        bool live = w[q] != kNone;
        const uint32_t wq = live ? w[q] : 0u;
        // v is a larger neighbour of w (LDF: the degree decides first, R21)
        hi[q] = live && pv > ((uint64_t)weight_mix(wq ^ a.key) | (a.dg ? (uint64_t)__ldg(a.dg + wq) << 32 : 0ull));
        cv[q] = kNone;
        // dead side (max-min): v's scheduling side was free at the start of
        // this round, so every neighbour on that side was coloured in an
        // earlier round and its counts decide nothing any more -- no atomic
        // (skipside 0: v freed by its hi side, its larger neighbours are dead;
        // 1: by its lo side, its smaller ones).  Decrements to uncoloured
        // vertices are never skipped, so the schedule is unchanged.
        if (kSkipDead && !JP && live && skipside >= 0 && hi[q] == (skipside == 1)) {
            w[q] = kNone;
            live = false;
        }
#if GC_PACKED
        slot[q] = (live && a.nbig > 0) ? big_slot(wq) : -1;
        uint32_t *adr = slot[q] >= 0 ? a.big32 + 2 * slot[q] + (hi[q] ? 0 : 1) : a.cnt32 + wq;
        const uint32_t dec = (slot[q] < 0 && hi[q]) ? kDec32Hi : 0xFFFFFFFFu;
        old[q] = live ? atom_add_global32(adr, dec) : 2u;
#else
        slot[q] = -1;
        if (JP) {
            old[q] = hi[q] ? atom_add_global(a.cnt + wq, kDecHi) : 2ull;
            if (live && !hi[q] && (want_mex || want_set)) cv[q] = __ldcg(a.C + wq);
        } else {
            old[q] = live ? atom_add_global(a.cnt + wq, hi[q] ? kDecHi : kDecLo) : 2ull;
        }
#endif
    }
    if (JP && want_set) {  // Alg.4: colours of v's coloured neighbours (their rounds' colours)
#pragma unroll
        for (int q = 0; q < Q; ++q) {
            if (w[q] != kNone && !hi[q]) {
                const uint32_t r = cv[q];  // a larger neighbour: coloured in an earlier round
                if (r >= k) flag_error(a, 5, k, v);
                const uint32_t c = r + 1u == k ? stage().cprev : __ldcg(a.cr + r);
                if (c < 32u * kCSetWords) atomicOr(stage().cset + (c >> 5), 1u << (c & 31u));
                else atomicOr(a.B + (size_t)(k % 3u) * a.bwords + (c >> 5), 1u << (c & 31u));
            }
        }
    }
    if (JP && want_mex) {
#pragma unroll
        for (int q = 0; q < Q; ++q) {
            if (w[q] != kNone && !hi[q] && cv[q] == GC_UNC) {
                // a predecessor's colour not seen yet (relaxed rounds) or an uncoloured predecessor (error)
                if (a.jrel) cv[q] = jp_read_once(a, a.C + w[q], GC_UNC, k, v);
                else flag_error(a, 5, k, v);
            }
            const uint32_t c = cv[q];
            if (w[q] != kNone && !hi[q]) {
                if (WIDE) {
                    if (c < 1024u) atomicOr(sbits + (c >> 5), 1u << (c & 31u));
                } else if (c < 64u) {
                    *mask |= 1ull << c;
                }
            }
        }
    }
    if (GC_PROF_UNIT && tprof) {
#pragma unroll
        for (int q = 0; q < Q; ++q) asm volatile("" ::"l"((unsigned long long)old[q]));
        tprof[1] = clock64();
    }
    bool fresh[Q];
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        fresh[q] = false;
        if (w[q] != kNone) {
            ++nvis;
            uint32_t side, other;
            if (!GC_PACKED) {
                side = hi[q] ? (uint32_t)(old[q] >> 32) : (uint32_t)old[q];
                other = hi[q] ? (uint32_t)old[q] : (uint32_t)(old[q] >> 32);
            } else if (slot[q] < 0) {
                side = hi[q] ? (uint32_t)old[q] >> 16 : (uint32_t)old[q] & 0xFFFFu;
                other = hi[q] ? (uint32_t)old[q] & 0xFFFFu : (uint32_t)old[q] >> 16;
            } else {  // big vertex: a side reaching zero claims the flag (rare)
                side = old[q];
                other = 1u;
                if (side == 1u) other = atom_or_global(a.big32 + 2 * kHTab + slot[q], 1u) ? 0u : 1u;
            }
            if (side == 1u) {
                if (other != 0u) fresh[q] = true;        // first side freed: schedule w
                else if (!hi[q]) a.Zlo[w[q]] = k + 1u;   // lo freed second (read after the rounds)
            } else if (side == 0u) {
                flag_error(a, 4, k, w[q]);  // count underflow: adjacency not symmetric
            }
        }
    }
    if (!JP && kEagerFresh) {
        // max-min: the warp schedules the neighbours it freed itself, right
        // after its unit (their row offsets loaded together), so the block
        // has no separate fresh step at the end of the round
        int64_t rsq[Q], req[Q];
#pragma unroll
        for (int q = 0; q < Q; ++q) {
            rsq[q] = fresh[q] ? __ldg(a.ro + w[q]) : 0;
            req[q] = fresh[q] ? __ldg(a.ro + w[q] + 1) : 0;
        }
#pragma unroll
        for (int q = 0; q < Q; ++q)
            if (__any_sync(kFull, fresh[q]))
                schedule_rows_slow<JP>(a, fresh[q], w[q], rsq[q], req[q] - rsq[q], kFirst | (hi[q] ? 0u : kLoSide));
        return;
    }
    // (rare) newly scheduled neighbours go to the block's fresh list; their
    // rows are fetched once per block at the end of the round (schedule_fresh)
    // instead of one dependent load per q here
    bool ovf[Q];
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        ovf[q] = false;
        if (fresh[q]) {
#if GC_EAGER_RO
            const longlong2 r = make_longlong2(a.ro[w[q]], a.ro[w[q] + 1]);
#else
            // its row offsets are loaded at the end of the round: start the
            // HBM -> L2 transfer now
            if (!GC_NO_PF_RO) asm volatile("prefetch.global.L2 [%0];" ::"l"(a.ro + w[q]));
#endif
            const unsigned pos = atomicAdd(&stage().nf, 1u);
            if (pos < (unsigned)kStF) {
                stage().fresh[pos] = make_uint2(w[q], hi[q] ? 0u : kLoSide);
#if GC_EAGER_RO
                stage().fro[pos] = r;
#endif
            } else {
                ovf[q] = true;
            }
        }
    }
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        if (__any_sync(kFull, ovf[q])) {  // shared list full: schedule here
            int64_t rs = 0, re = 0;
            if (ovf[q]) {
                rs = a.ro[w[q]];
                re = a.ro[w[q] + 1];
            }
            schedule_rows_slow<JP>(a, ovf[q], w[q], rs, re - rs, kFirst | (hi[q] ? 0u : kLoSide));
        }
    }
}

// MH (multi-hash, H weight functions, R8): walk the row of v coloured in
// round k; per entry w and per j decrement hi_j(w) or lo_j(w).  A side (j, s)
// reaching zero is free from round k+1: it records the code
// (k+1) << 5 | j << 1 | (s == hi) with atomicMin in Zlo[w], so Zlo[w] ends up
// holding w's decision -- its first free round, the smallest j free then, the
// min colour if that j's lo side is free (R8, R9) -- and sides freed in
// later rounds never override it.  The atomicMin that replaces kNever
// schedules w (exactly one per vertex).
template <int Q>
__device__ __forceinline__ void walk_mh(const CArgs &a, uint32_t v, int64_t e, int64_t end, int stride,
                                        uint32_t k, uint32_t &nvis, uint32_t zdec = kNever) {
    uint32_t w[Q];
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        const int64_t eq = e + (int64_t)q * stride;
        w[q] = (v != kNone && eq < end) ? __ldcs(a.ci + eq) : kNone;
    }
    const int H = a.H;
    if (kSkipDead && v != kNone && zdec != kNever) {
        // dead side (walk()): v's decision code names the weight function j
        // and the side of v that was free under it -- every neighbour on that
        // side is coloured, so none of its H counts needs a decrement
        const uint32_t js = (zdec >> 1) & 15u;
        const bool hifree = (zdec & 1u) != 0u;
        const uint32_t pvs = weight_mix(v ^ a.mkeys[js]);
#pragma unroll
        for (int q = 0; q < Q; ++q)
            if (w[q] != kNone && (pvs > weight_mix(w[q] ^ a.mkeys[js])) != hifree) w[q] = kNone;
    }
    if (GC_SKIP_COLOURED) {
        uint32_t mb[Q];
#pragma unroll
        for (int q = 0; q < Q; ++q) mb[q] = w[q] != kNone ? __ldcg(a.M + (w[q] >> 5)) : 0u;
#pragma unroll
        for (int q = 0; q < Q; ++q)
            if (w[q] != kNone && !((mb[q] >> (w[q] & 31u)) & 1u)) w[q] = kNone;
    }
    bool fresh[Q];
#pragma unroll
    for (int q = 0; q < Q; ++q) fresh[q] = false;
    if (H <= 4) {
        // H <= 4: the atomics of 4 entries x H weights are in flight together
        uint32_t pv[4];
#pragma unroll
        for (int j = 0; j < 4; ++j) pv[j] = j < H ? weight_mix(v ^ a.mkeys[j]) : 0u;
#pragma unroll
        for (int q0 = 0; q0 < Q; q0 += 4) {
            unsigned long long old[4][4];
            bool hi[4][4];
#pragma unroll
            for (int qq = 0; qq < 4; ++qq) {
                const int q = q0 + qq;
                if (q < Q && w[q] != kNone) {
#pragma unroll
                    for (int j = 0; j < 4; ++j) {
                        if (j < H) {
                            hi[qq][j] = pv[j] > weight_mix(w[q] ^ a.mkeys[j]);
                            old[qq][j] = atom_add_global(a.cnt + (size_t)w[q] * H + j, hi[qq][j] ? kDecHi : kDecLo);
                        }
                    }
                }
            }
#pragma unroll
            for (int qq = 0; qq < 4; ++qq) {
                const int q = q0 + qq;
                if (q < Q && w[q] != kNone) {
                    ++nvis;
#pragma unroll
                    for (int j = 0; j < 4; ++j) {
                        if (j < H) {
                            const uint32_t side = hi[qq][j] ? (uint32_t)(old[qq][j] >> 32) : (uint32_t)old[qq][j];
                            if (side == 1u) {
                                const uint32_t code = ((k + 1u) << 5) | ((uint32_t)j << 1) | (hi[qq][j] ? 1u : 0u);
                                if (atomicMin(a.Zlo + w[q], code) == kNever) fresh[q] = true;
                            } else if (side == 0u) {
                                flag_error(a, 4, k, w[q]);
                            }
                        }
                    }
                }
            }
        }
    } else {
        // H > 4: per entry, the weights in groups of 4 (4 atomics in flight)
#pragma unroll
        for (int q = 0; q < Q; ++q) {
            if (w[q] == kNone) continue;
            ++nvis;
            unsigned long long *cw = a.cnt + (size_t)w[q] * H;
            for (int j0 = 0; j0 < H; j0 += 4) {
                unsigned long long old[4];
                bool hi[4];
#pragma unroll
                for (int jj = 0; jj < 4; ++jj) {
                    const int j = j0 + jj;
                    if (j < H) {
                        hi[jj] = weight_mix(v ^ a.mkeys[j]) > weight_mix(w[q] ^ a.mkeys[j]);
                        old[jj] = atom_add_global(cw + j, hi[jj] ? kDecHi : kDecLo);
                    }
                }
#pragma unroll
                for (int jj = 0; jj < 4; ++jj) {
                    const int j = j0 + jj;
                    if (j < H) {
                        const uint32_t side = hi[jj] ? (uint32_t)(old[jj] >> 32) : (uint32_t)old[jj];
                        if (side == 1u) {
                            const uint32_t code = ((k + 1u) << 5) | ((uint32_t)j << 1) | (hi[jj] ? 1u : 0u);
                            if (atomicMin(a.Zlo + w[q], code) == kNever) fresh[q] = true;
                        } else if (side == 0u) {
                            flag_error(a, 4, k, w[q]);
                        }
                    }
                }
            }
        }
    }
    bool ovf[Q];
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        ovf[q] = false;
        if (fresh[q]) {
            asm volatile("prefetch.global.L2 [%0];" ::"l"(a.ro + w[q]));
            const unsigned pos = atomicAdd(&stage().nf, 1u);
            if (pos < (unsigned)kStF) {
                stage().fresh[pos] = make_uint2(w[q], 0u);
#if GC_EAGER_RO
                stage().fro[pos] = make_longlong2(a.ro[w[q]], a.ro[w[q] + 1]);
#endif
            }
            else ovf[q] = true;
        }
    }
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        if (__any_sync(kFull, ovf[q])) {
            int64_t rs = 0, re = 0;
            if (ovf[q]) {
                rs = a.ro[w[q]];
                re = a.ro[w[q] + 1];
            }
            schedule_rows_slow<false>(a, ovf[q], w[q], rs, re - rs, kFirst);
        }
    }
}

// The colour of v in its scheduled round k from its decision word z = Zlo[v]
// (max-min: min 2k+1 if the lo side is free at the start of round k -- the
// item's lo flag or a lo-freed-second stamp <= k --, else max 2k, Alg.5
// L37-42, R9; MH: the decision code).  The word is loaded
// when the item starts and consumed after the walk, so the walk's loads do
// not wait for it (a round's decision words are final at its start: words
// written during round k carry round k+1 and never change a round-k colour).
template <bool MH>
__device__ __forceinline__ void colour_fin(const CArgs &a, uint32_t v, uint32_t lf, uint32_t k, uint32_t z) {
    if (MH) {
        if ((z >> 5) != k) flag_error(a, 8, k, v);
        a.C[v] = 2u * (k * (uint32_t)a.H + ((z >> 1) & 15u)) + ((z & 1u) ? 0u : 1u);
    } else {
        a.C[v] = 2u * k + (((lf & kLoSide) || z <= k) ? 1u : 0u);
    }
    clear_status(a, v);
    atomicAdd(&stage().colored, 1u);
}


// Whole block, end of a round: stage the items of the vertices on the fresh
// list -- one THREAD per fresh vertex (row offsets in one dependent step),
// then the segments of all long rows written by the whole block.  An SL
// overflow, a long row that does not fit the staged WL buffer and a long-row
// list overflow go straight to the global lists (rare).
template <bool JP>
__device__ __forceinline__ void schedule_fresh(const CArgs &a, int64_t *prs = nullptr,
                                               unsigned long long t_round = 0) {
    Stage &st = stage();
    if (threadIdx.x == 0) st.nlong = 0;
    __syncthreads();
    if (prs && threadIdx.x == 0) {  // PROF: this block's units are done
        const unsigned long long dt = gtimer() - t_round;
        red_max(prs + 7, dt);
        if (!GC_PROF_UNIT && !GC_PROF_FRESH) red_max(prs + 9, ~dt);  // min via ~
        if (!GC_PROF_UNIT) red_max(prs + 13, (unsigned long long)st.nf);
        st.t_fs = gtimer();
    }
    const unsigned nf = min(st.nf, (unsigned)kStF);
    for (unsigned t = threadIdx.x; t < nf; t += blockDim.x) {
        const uint2 f = st.fresh[t];
#if GC_EAGER_RO
        const int64_t rs = st.fro[t].x, re = st.fro[t].y;
#else
        const int64_t rs = a.ro[f.x], re = a.ro[f.x + 1];
#endif
        const int64_t len = re - rs;
        if (GC_PROF_FRESH && prs) {  // this thread's row offsets are in
            asm volatile("" ::"l"(len));
            red_max(prs + 14, gtimer() - t_round);
        }
        const uint32_t fl = kFirst | f.y;
        if (len <= kShortMax) {
            Item it;
            it.v = f.x;
            it.lf = (uint32_t)len | fl;
            it.e0 = rs;
            if (len > 0) {  // the row walked next round: HBM -> L2 now (<= 2 lines)
                if (!GC_NO_PF_CI) asm volatile("prefetch.global.L2 [%0];" ::"l"(a.ci + rs));
                if (!GC_NO_PF_CI) asm volatile("prefetch.global.L2 [%0];" ::"l"(a.ci + re - 1));
            }
            const unsigned pos = atomicAdd(&st.n[0], 1u);
            if (pos < (unsigned)kStS) {
                st.s[pos] = it;
            } else {
                const unsigned long long at = st.nbase[0] + rw_field(atom_add_global(st.rw, 1ull), 0);
                if (at < a.sl_cap) gput(a.SL + grp_base(a, 0) + at, it);
                else flag_error(a, 1, 0, f.x);
            }
        } else {
            if (JP && a.jpv == 1) jp_slot_init(a, f.x, len);
            const uint32_t nseg = (uint32_t)((len + kSeg - 1) / kSeg);
            const unsigned sb = atomicAdd(&st.n[1], nseg);
            int64_t dst;
            if (sb + nseg <= (unsigned)kStW) {
                dst = (int64_t)sb;
            } else {
                // does not fit: global slots; staged slots [sb, kStW) become holes
                for (unsigned h = sb; h < (unsigned)kStW && h < sb + nseg; ++h) st.w[h].v = kNone;
                dst = ~(int64_t)(st.nbase[1] + rw_field(atom_add_global(st.rw, rw_add(nseg, 1)), 1));
            }
            // rows of <= kInlineSeg segments: this thread writes them now; longer
            // ones are expanded after the block barrier, one warp per row
            const unsigned li = nseg <= kInlineSeg ? (unsigned)kLongMax : atomicAdd(&st.nlong, 1u);
            if (li < (unsigned)kLongMax) {
                st.lng[li].rs = rs;
                st.lng[li].dst = dst;
                st.lng[li].w = f.x;
                st.lng[li].len = (uint32_t)len;
                st.lng[li].flags = fl;
            } else {  // short enough, or the long-row list is full: this thread writes them
                for (uint32_t q = 0; q < nseg; ++q) {
                    Item si;
                    si.v = f.x;
                    si.e0 = rs + (int64_t)q * kSeg;
                    si.lf = (uint32_t)min((int64_t)kSeg, len - (int64_t)q * kSeg) | ((q == 0 || (JP && a.jpv == 1)) ? fl : (fl & kLoSide));
                    if (dst >= 0) st.w[dst + q] = si;
                    else gput(a.WL + grp_base(a, 1) + ~dst + q, si);
                }
            }
        }
    }
    __syncthreads();
    if (GC_PROF_FRESH && prs && threadIdx.x == 0) red_max(prs + 15, gtimer() - t_round);
    const unsigned nl = min(st.nlong, (unsigned)kLongMax);
    for (unsigned r = threadIdx.x >> 5; r < nl; r += blockDim.x >> 5) {  // a warp per long row
        const Stage::Long L = st.lng[r];
        const uint32_t nseg = (L.len + kSeg - 1) / kSeg;
        for (uint32_t q = lane_id(); q < nseg; q += 32) {
            Item si;
            si.v = L.w;
            si.e0 = L.rs + (int64_t)q * kSeg;
            si.lf = (uint32_t)min((int64_t)kSeg, (int64_t)L.len - (int64_t)q * kSeg) | ((q == 0 || (JP && a.jpv == 1)) ? L.flags : (L.flags & kLoSide));
            if (L.dst >= 0) st.w[L.dst + q] = si;
            else gput(a.WL + grp_base(a, 1) + ~L.dst + q, si);
            if (GC_PREFETCH_WL) {  // the segment walked next round: HBM -> L2 now
                const uint32_t ln = si.lf & kLenMask;
                for (uint32_t o = 0; o < ln; o += 32) asm volatile("prefetch.global.L2 [%0];" ::"l"(a.ci + si.e0 + o));
            }
        }
    }
}

// JP, whole warp converged: this long-row segment of v has put its
// predecessors' colours into the warp's window `sb`; merge it into v's slot
// and retire its entries; the segment that retires the last entry computes
// the mex and colours v (first-fit, R10).
__device__ __noinline__ uint32_t jp_mex_rescan(const CArgs &a, uint32_t v, uint64_t pv, uint32_t *sb);

__device__ __forceinline__ void jp_segment_done(const CArgs &a, uint32_t v, uint32_t len, uint64_t pv,
                                                uint32_t *sb, uint32_t k, int64_t deg) {
    const unsigned lane = lane_id();
    __syncwarp();
    const uint32_t slot = a.jrel ? jp_read_once(a, a.Zlo + v, kNever, k, v) : __ldcg(a.Zlo + v);
    uint32_t *S = a.jslot + (size_t)slot * kSlotWords;
    const uint32_t word = sb[lane];
    if (word) atomicOr(S + lane, word);
    __threadfence();
    __syncwarp();
    uint32_t last = 0;
    if (lane == 0) {
        uint32_t old;
        if (a.jrel) {  // count up from the host's zero: the segment that completes the row is last
            asm volatile("atom.acq_rel.gpu.global.add.u32 %0, [%1], %2;"
                         : "=r"(old) : "l"(S + 32), "r"(len) : "memory");
            last = (int64_t)old + len == deg ? 1u : 0u;
            if ((int64_t)old + len > deg) flag_error(a, 7, k, v);
        } else {
            asm volatile("atom.acq_rel.gpu.global.add.u32 %0, [%1], %2;"
                         : "=r"(old) : "l"(S + 32), "r"(0u - len) : "memory");
            last = old == len ? 1u : 0u;
            if (old < len) flag_error(a, 7, k, v);
        }
    }
    last = __shfl_sync(kFull, last, 0);
    if (!last) return;
    __threadfence();
    const uint32_t bw = __ldcg(S + lane);
    const unsigned nf = __ballot_sync(kFull, bw != 0xFFFFFFFFu);
    uint32_t mex;
    if (nf) {
        const int f = __ffs(nf) - 1;
        mex = 32u * (uint32_t)f + (uint32_t)(__ffs(~__shfl_sync(kFull, bw, f)) - 1);
    } else {
        mex = jp_mex_rescan(a, v, pv, sb);
    }
    if (lane == 0) {
        a.C[v] = mex;
        atomicAdd(&stage().colored, 1u);
    }
}

// mex >= kMexWin (a vertex with >= 1024 predecessors of distinct colours):
// the warp rescans the row for successive 1024-colour windows (rare).
__device__ __noinline__ uint32_t jp_mex_rescan(const CArgs &a, uint32_t v, uint64_t pv, uint32_t *sb) {
    const unsigned lane = lane_id();
    const int64_t rs = a.ro[v], re = a.ro[v + 1];
    for (uint32_t b = kMexWin;; b += kMexWin) {
        __syncwarp();
        sb[lane] = 0u;
        __syncwarp();
        for (int64_t e = rs + lane; e < re; e += 32) {
            const uint32_t u = a.ci[e];
            if (prio_key(a, u) > pv) {
                const uint32_t c = (a.jrel ? jp_read_once(a, a.C + u, GC_UNC, 0u, v) : __ldcg(a.C + u)) - b;
                if (c < kMexWin) atomicOr(sb + (c >> 5), 1u << (c & 31u));
            }
        }
        __syncwarp();
        const uint32_t bw = sb[lane];
        const unsigned nf = __ballot_sync(kFull, bw != 0xFFFFFFFFu);
        if (nf) {
            const int f = __ffs(nf) - 1;
            return b + 32u * (uint32_t)f + (uint32_t)(__ffs(~__shfl_sync(kFull, bw, f)) - 1);
        }
    }
}

// Alg.4, whole block at the top of round k (after the grid barrier): the
// previous round's frontier colour = the smallest colour absent from the set
// its walks collected (R15); block 0 publishes it in cr[k-1] and clears the
// set that round k+1 will fill (its last reader was round k-1's top).
__device__ void jp4_round_top(const CArgs &a, uint32_t k, bool publisher) {
    Stage &st = stage();
    if (k > 0) {
        const uint32_t *S = a.B + (size_t)((k - 1u) % 3u) * a.bwords;
        const uint32_t W = min(a.bwords, (k - 1u) / 32u + 2u);
        if (threadIdx.x == 0) st.cmin = 0xFFFFFFFFu;
        __syncthreads();
        for (uint32_t w = threadIdx.x; w < W; w += blockDim.x) {
            const uint32_t x = __ldcg(S + w);
            if (x != 0xFFFFFFFFu) atomicMin(&st.cmin, 32u * w + (uint32_t)(__ffs(~x) - 1));
        }
        __syncthreads();
        if (threadIdx.x == 0) {
            st.cprev = st.cmin != 0xFFFFFFFFu ? st.cmin : 32u * W;
            if (publisher) a.cr[k - 1] = st.cprev;
        }
    }
    if (blockIdx.x == 0) {
        uint32_t *S2 = a.B + (size_t)((k + 1u) % 3u) * a.bwords;
        const uint32_t W2 = min(a.bwords, k / 32u + 3u);
        for (uint32_t w = threadIdx.x; w < W2; w += blockDim.x) S2[w] = 0u;
    }
    __syncthreads();
}

// 8-lane groups: OR of the group's masks
__device__ __forceinline__ unsigned long long group8_or(unsigned long long m) {
    m |= __shfl_xor_sync(kFull, m, 1);
    m |= __shfl_xor_sync(kFull, m, 2);
    m |= __shfl_xor_sync(kFull, m, 4);
    return m;
}

template <bool PROF, bool JP, bool MH>
// __grid_constant__: helpers take `const CArgs &`; without it the reference
// to a kernel parameter forces a per-thread local copy of CArgs (272 B of
// stack, every field access an LDL through L1): 31.1 -> 28.7 ms on R-MAT s24.
__global__ void __launch_bounds__((threads_for<JP, MH>()), 1) k_count_persistent(const __grid_constant__ CArgs a) {
    const unsigned lane = lane_id();
    const unsigned long long gtid = (unsigned long long)blockIdx.x * blockDim.x + threadIdx.x;
    const unsigned long long nthreads = (unsigned long long)gridDim.x * blockDim.x;
    const unsigned long long gwarp = gtid >> 5, nwarps = nthreads >> 5;
    const int64_t n = a.n;
    // max-min: rounds k >= 1 end with relaxed arrivals; the colours written
    // in the rounds are provisional (max unless the item's side is lo) and
    // the lo-freed-second stamps are applied after the rounds (final pass)
    constexpr bool kRelax = kRelaxedArrive && !JP && !MH;
    // relaxed rounds at run time: max-min always, JP for Luby and Alg.2 (a.jrel:
    // the values a later round reads are read until written, jp_read_once)
    const bool relax = kRelax || (JP && a.jrel);
    uint32_t nvis = 0;
    unsigned long long nvis_tot = 0, t_rounds = 0;
    unsigned long long t0 = PROF ? gtimer() : 0ull;
    {
        Stage &st = stage();
        if (threadIdx.x < 2) st.n[threadIdx.x] = 0;
        if (threadIdx.x < 2) st.nd[threadIdx.x] = 0;
        if (threadIdx.x == 0) st.colored = 0;
        if (threadIdx.x == 0) st.vis = 0;
        if (threadIdx.x == 0) st.nf = 0;
#if GC_PACKED
        for (int i = threadIdx.x; i < kHTab; i += blockDim.x) st.htab[i] = kNone;
#endif
        for (int i = threadIdx.x; i < kCSetWords; i += blockDim.x) st.cset[i] = 0u;
        __syncthreads();
#if GC_PACKED
        if (threadIdx.x == 0) {
            for (int i = 0; i < a.nbig; ++i) {
                const uint32_t v = a.big[i];
                unsigned h = hslot(v);
                while (st.htab[h] != kNone) h = (h + 1) & (kHTab - 1);
                st.htab[h] = v;
            }
        }
#endif
        // init appends round 0's items to slot 0 at position 0; its colourings
        // count for round 0 (so the "next round" targets are round 0's here)
        if (threadIdx.x == 0) {
            st.rw = round_word(a, 0, (int)(blockIdx.x % kNG));  // round 0's word
            st.tg_a = tag_a(a.epoch, 0u);
            st.tg_b = tag_b(a.epoch, 0u);
            st.nbase[0] = st.nbase[1] = 0ull;
            st.ccol = a.ctr + cK;
        }
        __syncthreads();
    }
    // ---------------------------------------------------- init = round 0
    // N_0 = n (written here: a colouring whose round 0 walks no row ends
    // before the round loop's bookkeeping)
    if (gtid == 0 && a.nk_cap > 0) a.nk[0] = n;
    // lane per vertex: a zero count colours v in round 0 (min wins, R9).  The
    // count word and the row offsets of kInitU batches of 32 vertices are
    // loaded together up front (independent loads: the phase is a stream)
    constexpr int kInitU = 4;
    // max-min (kInit2): a first pass counts the block's round-0 items, ONE
    // atomic per block reserves them, and the second pass writes each item
    // straight to its slot -- instead of millions of items spilling from the
    // block's staging through one round-word atomic per warp append
    constexpr bool kInit2 = kInitTwoPass && !JP && !MH && !GC_PACKED && kNG == 1;
    unsigned long long ib0 = 0, ib1 = 0;  // (kInit2) the block's first SL / WL slot of round 0
    if (kInit2) {
        // (the same vertices per warp as the second pass below: kInitU batches,
        // their count words and offsets loaded together up front)
        for (unsigned long long bb = gwarp * 32 * kInitU; bb < (unsigned long long)n; bb += nwarps * 32 * kInitU) {
          unsigned long long cq[kInitU];
          int64_t lq[kInitU];
#pragma unroll
          for (int b = 0; b < kInitU; ++b) {
            const unsigned long long vv = bb + 32ull * b + lane;
            const bool ok = vv < (unsigned long long)n;
            cq[b] = ok ? __ldcg(a.cnt + vv) : 0x100000001ull;
            lq[b] = ok ? __ldg(a.ro + vv + 1) - __ldg(a.ro + vv) : 0;
          }
#pragma unroll
          for (int b = 0; b < kInitU; ++b) {
            const int64_t len = lq[b];
            // (rows without entries: the count word is not written, and no item)
            const bool zero = len > 0 && ((uint32_t)(cq[b] >> 32) == 0u || (uint32_t)cq[b] == 0u);
            const unsigned nsl = __popc(__ballot_sync(kFull, zero && len <= kShortMax));
            const unsigned nwl = __reduce_add_sync(kFull, (zero && len > kShortMax) ? (unsigned)((len + kSeg - 1) / kSeg) : 0u);
            if (lane == 0) {
                if (nsl) atomicAdd(&stage().nd[0], nsl);
                if (nwl) atomicAdd(&stage().nd[1], nwl);
            }
          }
        }
        __syncthreads();
        Stage &st = stage();
        if (threadIdx.x == 0) {
            const unsigned long long t0i = st.nd[0], t1i = st.nd[1];
            const unsigned long long rv = (t0i || t1i) ? atom_add_global(st.rw, rw_add(t0i, 0) + rw_add(t1i, 1)) : 0ull;
            const unsigned long long r0 = rw_field(rv, 0), r1 = rw_field(rv, 1);
            if (r0 + t0i > kMSL || r1 + t1i > kMWL) flag_error(a, 9, 0, 0);
            if (r0 + t0i > a.sl_cap || r1 + t1i > a.wl_cap) flag_error(a, 2, 0, 0);
            st.base[0] = r0;
            st.base[1] = r1;
            st.nd[0] = st.nd[1] = 0;  // now the position counters
        }
        __syncthreads();
        ib0 = st.base[0];
        ib1 = st.base[1];
    }
    for (unsigned long long base0 = gwarp * 32 * kInitU; base0 < (unsigned long long)n;
         base0 += nwarps * 32 * kInitU) {
      unsigned long long cpre[kInitU];
      int64_t rspre[kInitU], repre[kInitU];
#pragma unroll
      for (int b = 0; b < kInitU; ++b) {
        const unsigned long long vv = base0 + 32ull * b + lane;
        const bool ok = !MH && vv < (unsigned long long)n;
        cpre[b] = ok ? __ldcs(a.cnt + vv) : 0x100000001ull;
        rspre[b] = ok ? __ldg(a.ro + vv) : 0;
        repre[b] = ok ? __ldg(a.ro + vv + 1) : 0;
      }
#pragma unroll
      for (int b = 0; b < kInitU; ++b) {
        const unsigned long long base = base0 + 32ull * b;
        if (base >= (unsigned long long)n) break;
        const uint32_t v = (uint32_t)(base + lane);
        const bool valid = (int64_t)(base + lane) < n;
        uint32_t hi = 1u, lo = 1u, code = kNever;
        if (MH) {
            // round 0: the smallest j with a free side, its min side first (R8, R9)
            for (int j = 0; valid && j < a.H; ++j) {
                const unsigned long long c = a.cnt[(size_t)v * a.H + j];
                if ((uint32_t)c == 0u) code = min(code, (uint32_t)j << 1);
                else if ((uint32_t)(c >> 32) == 0u) code = min(code, ((uint32_t)j << 1) | 1u);
            }
        } else if (rspre[b] == repre[b]) {
            hi = 0u;  // no entries: the counting pass does not write the count word
            lo = JP ? 1u : 0u;
        } else {
            const unsigned long long c = cpre[b];
            hi = (uint32_t)(c >> 32);
            lo = (uint32_t)c;
        }
        const bool zero = valid && (MH ? code != kNever : (hi == 0u || lo == 0u));
        int64_t rs = 0, re = 0;
        if (valid) {
            const int sl = (GC_PACKED && a.nbig > 0) ? big_slot(v) : -1;
            if (!GC_PACKED || MH) {
            } else if (sl < 0) {
                a.cnt32[v] = (hi << 16) | lo;  // deg <= kPackMax
            } else {
                a.big32[2 * sl] = hi;
                a.big32[2 * sl + 1] = lo;
                a.big32[2 * kHTab + sl] = (hi == 0u || lo == 0u) ? 1u : 0u;
            }
            if (MH) {
                a.Zlo[v] = code;  // round 0's decision (not kNever: never rescheduled)
                a.C[v] = zero ? 2u * (code >> 1) + ((code & 1u) ? 0u : 1u) : GC_UNC;
            } else {
                if (!JP || a.jrel) a.Zlo[v] = kNever;
                a.C[v] = zero ? (lo == 0u ? 1u : 0u) : GC_UNC;
            }
            if (zero) {
                rs = MH ? a.ro[v] : rspre[b];
                re = MH ? a.ro[v + 1] : repre[b];
            }
        }
        const unsigned word = __ballot_sync(kFull, zero);
        if (GC_SKIP_COLOURED && !JP) {
            // status word of these 32 vertices: uncoloured after round 0's decisions
            const unsigned live = __ballot_sync(kFull, valid && !zero);
            if (lane == 0) a.M[base >> 5] = live;
        }
        if (lane == 0 && word) atomicAdd(&stage().colored, (unsigned)__popc(word));
        // walked in round 0 (the free side's flag: its neighbours, if any, are dead)
        if (kInit2) {
            const uint32_t fl = lo == 0u ? kLoSide : 0u;
            const int64_t len = re - rs;
            const bool sl = zero && len > 0 && len <= kShortMax;
            const unsigned msl = __ballot_sync(kFull, sl);
            if (msl) {
                unsigned p0 = 0;
                if (lane == (unsigned)(__ffs(msl) - 1)) p0 = atomicAdd(&stage().nd[0], (unsigned)__popc(msl));
                p0 = __shfl_sync(kFull, p0, __ffs(msl) - 1);
                if (sl) {
                    Item it;
                    it.v = v;
                    it.lf = (uint32_t)len | fl;
                    it.e0 = rs;
                    gput(a.SL + ib0 + p0 + __popc(msl & ((1u << lane) - 1u)), it);
                }
            }
            const bool lg = zero && len > kShortMax;
            const uint32_t nseg = lg ? (uint32_t)((len + kSeg - 1) / kSeg) : 0u;
            const unsigned pw = lg ? atomicAdd(&stage().nd[1], nseg) : 0u;
            unsigned lm = __ballot_sync(kFull, lg);
            while (lm) {  // the warp writes each long row's segments
                const int src = __ffs(lm) - 1;
                lm &= lm - 1;
                const uint32_t ww = __shfl_sync(kFull, v, src);
                const int64_t r0 = __shfl_sync(kFull, rs, src), ln = __shfl_sync(kFull, len, src);
                const uint32_t fs = __shfl_sync(kFull, fl, src), ns = __shfl_sync(kFull, nseg, src);
                const unsigned ps = __shfl_sync(kFull, pw, src);
                for (uint32_t q = lane; q < ns; q += 32) {
                    Item si;
                    si.v = ww;
                    si.e0 = r0 + (int64_t)q * kSeg;
                    si.lf = (uint32_t)min((int64_t)kSeg, ln - (int64_t)q * kSeg) | fs;
                    gput(a.WL + ib1 + ps + q, si);
                }
            }
        } else {
            schedule_rows<JP>(a, zero && re > rs, v, rs, re - rs, (!JP && !MH && lo == 0u) ? kLoSide : 0u);
        }
      }
    }
    if (kInit2) {  // (the items are written; the arrival below reserves none)
        __syncthreads();
        if (threadIdx.x == 0) stage().nd[0] = stage().nd[1] = 0;
    }
    stage_flush(a);
    if (!grid_barrier_rw(a, 0, 0, stage().rd)) return;
    if (PROF && gtid == 0) {
        const unsigned long long t = gtimer();
        a.ctr[cPhaseNs] = t - t0;
        t0 = t;
    }
    // ------------------------------------------------------------ rounds
    // work units of a round: WL items u < nw, then groups of 4 SL items; unit
    // u goes to block u % G, warp (u / G) % wpb of it (round-robin over SMs)
    const unsigned wpb = blockDim.x >> 5;
    const unsigned long long u_first =
        (unsigned long long)(threadIdx.x >> 5) * gridDim.x + blockIdx.x;
    unsigned long long sl0[kNG], wl0[kNG];  // per group: where round k's items start
#pragma unroll
    for (int gq = 0; gq < kNG; ++gq) sl0[gq] = wl0[gq] = 0;
    int64_t rem = n;                      // gtid 0 only: uncoloured at the round start
    uint32_t last = 0;                    // last round with a colouring
    uint32_t k = 0;
    for (;; ++k) {
        const unsigned long long t_round = PROF ? gtimer() : 0ull;
        const int cur = (int)(k % 3);
        // one thread per block reads the round's counters (2,368 warps reading
        // the same L2 line serialise in its slice) and sets the append targets
        // the round's item counts came with the barrier's last load (round
        // word); the trap flag is read every 32 rounds (a trap ends the
        // kernel at most 32 rounds later, grid-uniformly)
        if (threadIdx.x == 0) {
            Stage &st = stage();
            const int me = (int)(blockIdx.x % kNG);
            st.gn[0][0] = st.gn[1][0] = 0;
#pragma unroll
            for (int gq = 0; gq < kNG; ++gq) {
                const unsigned long long r_ns = rw_field(st.rd[gq], 0), r_nw = rw_field(st.rd[gq], 1);
                st.gn[0][gq + 1] = st.gn[0][gq] + r_ns;
                st.gn[1][gq + 1] = st.gn[1][gq] + r_nw;
                st.g0[0][gq] = sl0[gq];
                st.g0[1][gq] = wl0[gq];
                if (gq == me) {
                    st.nbase[0] = sl0[gq] + r_ns;
                    st.nbase[1] = wl0[gq] + r_nw;
                }
            }
            st.trap = (k & 31u) == 0u ? __ldcg(&a.ctr[cErr]) : 0ull;
            if (kDirectFlush && !MH) {  // (the last round's direct flush is done)
                st.n[0] = st.n[1] = 0;
                st.nd[0] = st.nd[1] = 0;
                st.nf = 0;
            }
            st.rw = round_word(a, (int)((k + 1) % 3), me);
            st.tg_a = tag_a(a.epoch, k + 1u);
            st.tg_b = tag_b(a.epoch, k + 1u);
            st.ccol = a.ctr + cK + 16 * cur;
        }
        __syncthreads();
        if (JP && a.jpv == 3) jp4_round_top(a, k, gtid == 0);
        const unsigned long long ns = stage().gn[0][kNG], nw = stage().gn[1][kNG];
        // words of round k+2 (their last reader: the barrier that ended round k-2)
        if (gtid == 0) {
#pragma unroll
            for (int gq = 0; gq < kNG; ++gq) *round_word(a, (int)((k + 2) % 3), gq) = 0ull;
        }
        if (stage().trap != 0ull) break;  // a trap fired (uniform: read after a barrier)
        if (ns == 0 && nw == 0) break;            // nothing scheduled: done
        if (k >= a.max_rounds) break;
        if (k > 0) last = k;  // every item of round k >= 1 colours (kFirst)
        if (PROF && gtid == 0 && (int64_t)k < a.nk_cap) {
            a.rstat[16 * k + 0] = (int64_t)ns;
            a.rstat[16 * k + 1] = (int64_t)nw;
        }
        int64_t *prs = (PROF && (int64_t)k < a.nk_cap) ? a.rstat + 16 * k : nullptr;
        if (prs && threadIdx.x == 0)
            red_max(prs + 6, gtimer() - t_round);
        // a large SL list (round 0: millions of mostly 1-4-entry rows) is
        // walked one row per LANE, so a warp has 32 rows in flight, not 4
        const bool lane_rows = ns > 16ull * nwarps;
        const unsigned long long units = nw + (lane_rows ? (ns + 31) / 32 : (ns + 3) / 4);
        for (unsigned long long u = u_first; u < units; u += nwarps) {
            const long long c_unit = PROF ? clock64() : 0;
            if (u < nw) {
                // longer rows: one <= kSeg-entry item per warp
                Item it = gget(a, round_item(a, 1, u), k);
                if (it.v == kNone) it.lf = 0;  // hole left by schedule_fresh
                const uint64_t pv = prio_key(a, it.v);
                if (JP && a.jpv != 1) {  // Alg.2 / Alg.4: the colour is the round (remapped for Alg.4)
                    if ((it.lf & kFirst) && lane == 0) {
                        a.C[it.v] = k;
                        atomicAdd(&stage().colored, 1u);
                    }
                    walk<kSeg / 32, true>(a, it.v, pv, it.e0 + lane, it.e0 + (it.lf & kLenMask), 32, k, nvis,
                                          nullptr, nullptr, false, a.jpv == 3);
                } else if (JP && (it.lf & kFirst)) {  // a segment of a row being coloured
                    uint32_t *sb = stage().wbits[threadIdx.x >> 5];
                    sb[lane] = 0u;
                    // (relaxed rounds: the row's length for the count-up completion, loaded now)
                    const int64_t dgv = a.jrel ? __ldg(a.ro + it.v + 1) - __ldg(a.ro + it.v) : 0;
                    __syncwarp();
                    walk<kSeg / 32, true, true>(a, it.v, pv, it.e0 + lane, it.e0 + (it.lf & kLenMask), 32, k,
                                                nvis, nullptr, sb, true);
                    jp_segment_done(a, it.v, it.lf & kLenMask, pv, sb, k, dgv);
                } else {
                    const bool cl = !JP && (it.lf & kFirst) && lane == 0;
                    const uint32_t z = (cl && !kRelax) ? __ldcg(a.Zlo + it.v) : kNever;
                    long long tp[3] = {0, 0, 0};
                    if (GC_PROF_UNIT && prs) {
                        asm volatile("" ::"l"(pv));
                        tp[2] = clock64();
                    }
                    if (MH)
                        walk_mh<kSeg / 32>(a, it.v, it.e0 + lane, it.e0 + (it.lf & kLenMask), 32, k, nvis,
                                           it.v != kNone ? __ldcg(a.Zlo + it.v) : kNever);
                    else
                        walk<kSeg / 32, JP>(a, it.v, pv, it.e0 + lane, it.e0 + (it.lf & kLenMask), 32, k, nvis,
                                            nullptr, nullptr, false, false, (GC_PROF_UNIT && prs) ? tp : nullptr,
                                            JP ? -1 : ((it.lf & kLoSide) ? 1 : 0));
                    if (cl) colour_fin<MH>(a, it.v, it.lf, k, z);
                    if (GC_PROF_UNIT && prs && !MH) {
                        // max over the warp's lanes of each stage's end (cycles since the unit start)
                        const unsigned mi = __reduce_max_sync(kFull, (unsigned)(tp[2] - c_unit));
                        const unsigned mc = __reduce_max_sync(kFull, (unsigned)(tp[0] - c_unit));
                        const unsigned ma = __reduce_max_sync(kFull, (unsigned)(tp[1] - c_unit));
                        if (lane == 0) {
                            red_max(prs + 12, mi);
                            red_max(prs + 14, mc);
                            red_max(prs + 15, ma);
                            red_add(prs + 11, mc);        // sum: unit start -> column ids in
                            red_add(prs + 9, ma - mc);    // sum: column ids -> atomics back
                        }
                    }
                }
            } else if (lane_rows) {
                // short rows: one per lane, 4 entries per step
                const unsigned long long idx = 32 * (u - nw) + lane;
                uint32_t v = kNone, len = 0;
                uint64_t pv = 0;
                int64_t e0 = 0;
                bool want = false, cl = false;
                uint32_t lf = 0, z = kNever;
                if (idx < ns) {
                    const Item it = gget(a, round_item(a, 0, idx), k);
                    v = it.v;
                    lf = it.lf;
                    len = it.lf & kLenMask;
                    e0 = it.e0;
                    pv = prio_key(a, v);
                    want = JP && a.jpv == 1 && (it.lf & kFirst);
                    if (JP && a.jpv != 1 && (it.lf & kFirst)) {
                        a.C[v] = k;
                        atomicAdd(&stage().colored, 1u);
                    }
                    cl = !JP && (it.lf & kFirst);
                    if (cl && !kRelax) z = __ldcg(a.Zlo + v);
                }
                unsigned long long mask = 0ull;
                const uint32_t zm = (MH && v != kNone) ? __ldcg(a.Zlo + v) : kNever;  // (MH: v's decision)
                for (uint32_t j = 0; __any_sync(kFull, j < len); j += 4) {
                    if (MH) walk_mh<4>(a, j < len ? v : kNone, e0 + j, e0 + len, 1, k, nvis, zm);
                    else walk<4, JP>(a, j < len ? v : kNone, pv, e0 + j, e0 + len, 1, k, nvis, &mask, nullptr, want,
                                     JP && a.jpv == 3, nullptr, JP ? -1 : ((lf & kLoSide) ? 1 : 0));
                }
                if (cl) colour_fin<MH>(a, v, lf, k, z);
                if (JP && want) {  // <= 32 predecessors: the mex is below 64
                    a.C[v] = (uint32_t)(__ffsll((long long)~mask) - 1);
                    atomicAdd(&stage().colored, 1u);
                }
            } else {
                // short rows: 4 per warp, 8 lanes each, 4 entries per lane
                const unsigned long long idx = 4 * (u - nw) + (lane >> 3);
                uint32_t v = kNone, len = 0;
                uint64_t pv = 0;
                int64_t e0 = 0;
                bool want = false, cl = false;
                uint32_t lf = 0, z = kNever;
                if (idx < ns) {
                    const Item it = gget(a, round_item(a, 0, idx), k);
                    v = it.v;
                    lf = it.lf;
                    len = it.lf & kLenMask;
                    e0 = it.e0;
                    pv = prio_key(a, v);
                    want = JP && a.jpv == 1 && (it.lf & kFirst);
                    if (JP && a.jpv != 1 && (it.lf & kFirst) && (lane & 7u) == 0u) {
                        a.C[v] = k;
                        atomicAdd(&stage().colored, 1u);
                    }
                    cl = !JP && (it.lf & kFirst) && (lane & 7u) == 0u;
                    if (cl && !kRelax) z = __ldcg(a.Zlo + v);
                }
                unsigned long long mask = 0ull;
                const uint32_t zm = (MH && v != kNone) ? __ldcg(a.Zlo + v) : kNever;  // (MH: v's decision)
                if (MH) walk_mh<4>(a, v, e0 + (lane & 7u), e0 + len, 8, k, nvis, zm);
                else walk<4, JP>(a, v, pv, e0 + (lane & 7u), e0 + len, 8, k, nvis, &mask, nullptr, want,
                                 JP && a.jpv == 3, nullptr, JP ? -1 : ((lf & kLoSide) ? 1 : 0));
                if (cl) colour_fin<MH>(a, v, lf, k, z);
                if (JP && a.jpv == 1) {
                    mask = group8_or(mask);
                    if (want && (lane & 7u) == 0u) {
                        a.C[v] = (uint32_t)(__ffsll((long long)~mask) - 1);
                        atomicAdd(&stage().colored, 1u);
                    }
                }
            }
            if (prs && lane == 0)
                red_max(prs + ((GC_PROF_UNIT && u >= nw) ? 13 : 10), (unsigned long long)(clock64() - c_unit));
        }
#pragma unroll
        for (int gq = 0; gq < kNG; ++gq) {
            sl0[gq] += rw_field(stage().rd[gq], 0);
            wl0[gq] += rw_field(stage().rd[gq], 1);
        }
        if (PROF) {
            const unsigned s = __reduce_add_sync(kFull, nvis);
            if (lane == 0 && s) atomicAdd(&stage().vis, s);
        }
        nvis_tot += nvis;  // (always: the count decrements issued, for the algorithmic bytes)
        nvis = 0;
        if (gtid == 0) {  // bookkeeping: uncoloured at the start of round k (off the round top)
            if (k > 0) {
                const int prv = (int)((k + 2) % 3);
                rem -= (int64_t)__ldcg(&a.ctr[cK + 16 * prv]);
                a.ctr[cK + 16 * prv] = 0ull;  // only gtid 0 reads these slots
            }
            if ((int64_t)k < a.nk_cap) a.nk[k] = rem;
            if (PROF && k > 0 && (int64_t)(k - 1) < a.nk_cap) a.rstat[16 * (k - 1) + 3] = a.nk[k - 1] - rem;
        }
        if (JP && a.jpv == 3) {  // the block's share of this round's colour set -> global
            __syncthreads();
            Stage &st = stage();
            const uint32_t wmax = min((uint32_t)kCSetWords, k / 32u + 2u);
            for (uint32_t w = threadIdx.x; w < wmax; w += blockDim.x) {
                const uint32_t x = st.cset[w];
                if (x) {
                    atomicOr(a.B + (size_t)(k % 3u) * a.bwords + w, x);
                    st.cset[w] = 0u;
                }
            }
        }
        if (kDirectFlush && !MH) {
            fresh_flush_direct<JP>(a, relax, prs, t_round);
        } else {
            if (!(kEagerFresh && !JP && !MH)) schedule_fresh<JP>(a, prs, t_round);
            stage_flush(a, prs, t_round, relax);
        }
        if (!grid_barrier_rw(a, k, (int)((k + 1) % 3), stage().rd, !relax)) return;
        if (PROF && gtid == 0) {
            const unsigned long long t = gtimer();
            if ((int64_t)k < a.nk_cap) a.rstat[16 * k + 4] = (int64_t)(t - t0);
            t_rounds += t - t0;
            t0 = t;
        }
    }
    (void)wpb;
    if (relax) {
        // one release / acquire barrier (every block's stamps and colours are
        // visible), then each colour of round k >= 1 that was written as the
        // max 2k becomes the min 2k+1 if v's lo side was freed second by
        // round k (Zlo[v] <= k: min wins, Alg.5 L37-42, R9); a stamp of a
        // later round never changes it.  The coloured vertices are counted
        // here (the completion check).
        __syncthreads();
        if (threadIdx.x == 0) {
            atom_add_release(a.ctr + cFin, 1ull);
            const unsigned long long t0f = gtimer();
            while (ld_acquire(a.ctr + cFin) < gridDim.x) {
                if (gtimer() - t0f > 4000000000ull) {
                    flag_error(a, 100, k, blockIdx.x);
                    break;
                }
            }
        }
        __syncthreads();
        uint32_t ncol = 0, cmax = 0;
        for (unsigned long long v = gtid; v < (unsigned long long)n; v += nthreads) {
            uint32_t c = __ldcg(a.C + v);
            if (c == GC_UNC) continue;
            ++ncol;
            if (!JP && (c & 1u) == 0u && __ldcg(a.Zlo + v) <= (c >> 1)) a.C[v] = (c |= 1u);
            cmax = max(cmax, c);
        }
        const unsigned s = __reduce_add_sync(kFull, ncol);
        if (lane == 0 && s) atomicAdd(&a.ctr[cCol], (unsigned long long)s);
        // the largest colour (the distinct-colour count sizes its set with it)
        const unsigned mx = __reduce_max_sync(kFull, cmax);
        if (lane == 0 && s) atomicMax(&a.ctr[cMaxC], (unsigned long long)mx + 1ull);
    }
    if (JP && a.jpv == 3) {
        // colours were round indices: C[v] <- colour of its round (the last
        // round's colour is this block's cprev; earlier ones are in cr)
        const uint32_t cp = stage().cprev;
        for (unsigned long long v = gtid; v < (unsigned long long)n; v += nthreads) {
            const uint32_t r = a.C[v];
            // (k == 0: only init's round-0 vertices, whose colour is mex of {} = 0)
            if (r != GC_UNC) a.C[v] = k == 0 ? 0u : r + 1u == k ? cp : __ldcg(a.cr + r);
        }
    }
    if (gtid == 0) {
        a.ctr[cRounds] = n > 0 ? last + 1 : 0;
        a.ctr[cIters] = k;
        // the colourings of round k-1 (init's for k == 0) not yet subtracted
        rem -= (int64_t)__ldcg(&a.ctr[cK + 16 * (k == 0 ? 0 : (int)((k + 2) % 3))]);
        if (!relax) a.ctr[cCol] = (unsigned long long)(n - rem);
        if (PROF) a.ctr[cPhaseNs + 1] = t_rounds;
    }
    {
        const unsigned long long s = __reduce_add_sync(kFull, (unsigned)nvis_tot);
        if (lane == 0 && s) atomicAdd(&a.ctr[cVis], s);
    }
}

// hi / lo counts of every vertex (round-0 state: everything is uncoloured),
// per weight function j < H (MH: the multi-hash variant; word v * H + j).
// A warp takes 32 consecutive vertices: rows <= 16 one lane each, rows up to
// kHubMin the whole warp (coalesced), longer rows go to the hub list.
struct CountKeys {
    uint32_t k[GC_MAX_HASHES];
    int H;
};

// LDF (dg != nullptr, H = 1): the key of R21, (degree, weight), decides
__device__ __forceinline__ uint64_t ckey(const uint32_t *dg, uint32_t v, uint32_t key) {
    const uint64_t w = weight_mix(v ^ key);
    return dg ? w | ((uint64_t)__ldg(dg + v) << 32) : w;
}

template <bool MH>
__global__ void __launch_bounds__(256) k_count(const int64_t *__restrict__ ro,
                                               const uint32_t *__restrict__ ci, int64_t n,
                                               CountKeys keys, unsigned long long *cnt,
                                               uint2 *hubs, unsigned long long *nhubs, int jp,
                                               const uint32_t *__restrict__ dg) {
    const unsigned lane = lane_id();
    const unsigned long long gw = ((unsigned long long)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const unsigned long long nw = ((unsigned long long)gridDim.x * blockDim.x) >> 5;
    const int H = MH ? keys.H : 1;
    for (unsigned long long base = gw * 32; base < (unsigned long long)n; base += nw * 32) {
        const int64_t v = (int64_t)(base + lane);
        const bool valid = v < n;
        int64_t rs = 0, re = 0;
        if (valid) {
            rs = ro[v];
            re = ro[v + 1];
        }
        const int64_t deg = re - rs;
        // rows of <= 16 entries: one lane each, as many steps as the warp's
        // longest such row (not always 16: most short rows have 1-4 entries)
        const bool lrow = valid && deg <= 16;
        const int dmax = (int)__reduce_max_sync(kFull, lrow ? (unsigned)deg : 0u);
        if (lrow) {
            uint32_t u[16];
#pragma unroll
            for (int q = 0; q < 16; ++q) u[q] = (q < dmax && q < deg) ? __ldcs(ci + rs + q) : 0u;
            for (int j = 0; j < H; ++j) {
                const uint32_t key = keys.k[j];
                const uint64_t pv = ckey(MH ? nullptr : dg, (uint32_t)v, key);
                uint32_t h = 0;
#pragma unroll
                for (int q = 0; q < 16; ++q)
                    if (q < dmax) h += (q < deg && ckey(MH ? nullptr : dg, u[q], key) > pv) ? 1u : 0u;
                cnt[(size_t)v * H + j] = ((unsigned long long)h << 32) | (unsigned long long)(jp ? 1 : deg - h);
            }
        }
        const bool big = valid && deg > kHubMin;
        if (big) {
            for (int j = 0; j < H; ++j) cnt[(size_t)v * H + j] = jp ? 1ull : 0ull;  // k_count_hub adds the chunks
            const int64_t nch = (deg + kHubChunk - 1) / kHubChunk;
            const unsigned long long b = atomicAdd(nhubs, (unsigned long long)nch);
            for (int64_t c = 0; c < nch; ++c)
                hubs[b + c] = make_uint2((uint32_t)v, (uint32_t)c);
        }
        unsigned mid = __ballot_sync(kFull, valid && deg > 16 && deg <= kHubMin);
        while (mid) {
            const int src = __ffs(mid) - 1;
            mid &= mid - 1;
            const int64_t r0 = __shfl_sync(kFull, rs, src), r1 = __shfl_sync(kFull, re, src);
            const uint32_t vs = (uint32_t)(base + src);
            for (int j = 0; j < H; ++j) {
                const uint32_t key = keys.k[j];
                const uint64_t p = ckey(MH ? nullptr : dg, vs, key);
                uint32_t h = 0;
                for (int64_t e = r0 + lane; e < r1; e += 128) {
                    uint32_t u[4];
#pragma unroll
                    for (int q = 0; q < 4; ++q) u[q] = e + 32 * q < r1 ? __ldcs(ci + e + 32 * q) : 0u;
#pragma unroll
                    for (int q = 0; q < 4; ++q)
                        h += (e + 32 * q < r1 && ckey(MH ? nullptr : dg, u[q], key) > p) ? 1u : 0u;
                }
                h = __reduce_add_sync(kFull, h);
                if (lane == (unsigned)src)
                    cnt[(size_t)v * H + j] =
                        ((unsigned long long)h << 32) | (unsigned long long)(jp ? 1 : deg - h);
            }
        }
    }
}

// Rows longer than kHubMin: one block per kHubChunk-entry chunk (the chunk
// list (v, c) was written by k_count); partial counts are added atomically.
template <bool MH>
__global__ void __launch_bounds__(256) k_count_hub(const int64_t *__restrict__ ro,
                                                   const uint32_t *__restrict__ ci, CountKeys keys,
                                                   unsigned long long *cnt, const uint2 *hubs,
                                                   const unsigned long long *nhubs, int jp,
                                                   const uint32_t *__restrict__ dg) {
    __shared__ uint32_t red[8];
    const unsigned long long nh = *nhubs;
    const int H = MH ? keys.H : 1;
    for (unsigned long long i = blockIdx.x; i < nh; i += gridDim.x) {
        const uint2 hc = hubs[i];
        const uint32_t v = hc.x;
        const int64_t rs = ro[v], re = ro[v + 1];
        const int64_t c0 = rs + (int64_t)hc.y * kHubChunk, c1 = min(re, c0 + (int64_t)kHubChunk);
        for (int j = 0; j < H; ++j) {
            const uint32_t key = keys.k[j];
            const uint64_t pv = ckey(MH ? nullptr : dg, v, key);
            uint32_t hcount = 0;
#pragma unroll 4
            for (int64_t e = c0 + threadIdx.x; e < c1; e += blockDim.x)
                hcount += ckey(MH ? nullptr : dg, __ldcs(ci + e), key) > pv ? 1u : 0u;
            hcount = __reduce_add_sync(kFull, hcount);
            if (lane_id() == 0) red[threadIdx.x >> 5] = hcount;
            __syncthreads();
            if (threadIdx.x == 0) {
                uint32_t t = 0;
                for (int w = 0; w < (int)(blockDim.x >> 5); ++w) t += red[w];
                const unsigned long long tot = (unsigned long long)(c1 - c0);
                atomicAdd(&cnt[(size_t)v * H + j], ((unsigned long long)t << 32) + (jp ? 0ull : tot - t));
            }
            __syncthreads();
        }
    }
}

// ------------------------------------------------ counting pass: warp tiles
// The counting pass is the one full read of the CSR (round 0's max / min test
// of Alg.5 for every vertex at once), written as an HBM stream: warp tile w
// is the kWE consecutive column ids [w kWE, +kWE), whatever the degree mix, so
// every load is a coalesced 16-byte vector and no block barrier is needed.  A
// lane takes kWQ consecutive entries (the next tile's are loaded before the
// current one is counted).  The rows of the tile are visited in chunks of 32
// (their offsets staged in the warp's shared slots); a lane finds the row of
// its next entry by binary search there and walks forward; per-row hi counts
// are summed in the warp's shared slots.  Rows inside the tile are written
// once, rows crossing a tile boundary (pre-set by k_count_zero) get one
// 64-bit atomic per tile.  Rows without entries are not written: the init
// phase of the rounds reads their zero degree from the offsets.
// crow[w] = the row of tile w's first entry (seed-independent, once per graph).
#ifndef GC_WQ
#define GC_WQ 16
#endif
constexpr int kWQ = GC_WQ;          // entries per lane
constexpr int kWE = 32 * kWQ;       // entries per warp tile
constexpr int kWT = 256;            // threads per block
constexpr int kTE = kWE;            // (tile granularity of crow / k_count_zero)

// crow[c] = last row r with ro[r] <= c * kTE (crow[0] = 0, crow[nch] = n - 1)
__global__ void k_chunk_rows(const int64_t *__restrict__ ro, int64_t n, int64_t nch, uint32_t *crow) {
    for (int64_t c = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; c <= nch;
         c += (int64_t)gridDim.x * blockDim.x) {
        if (c == 0 || c == nch) {
            crow[c] = c == 0 ? 0u : (uint32_t)(n - 1);
            continue;
        }
        const int64_t e = c * kTE;
        int64_t lo = 0, hi = n;  // ro[lo] <= e < ro[hi]
        while (hi - lo > 1) {
            const int64_t mid = (lo + hi) >> 1;
            if (ro[mid] <= e) lo = mid;
            else hi = mid;
        }
        crow[c] = (uint32_t)lo;
    }
}

// rows crossing a tile boundary start from zero (JP: lo pinned at 1)
__global__ void k_count_zero(const int64_t *__restrict__ ro, const uint32_t *__restrict__ crow, int64_t nch,
                             unsigned long long *cnt, int jp) {
    for (int64_t c = 1 + (int64_t)blockIdx.x * blockDim.x + threadIdx.x; c < nch;
         c += (int64_t)gridDim.x * blockDim.x) {
        const uint32_t r = crow[c];
        if (ro[r] < c * kTE) cnt[r] = jp ? 1ull : 0ull;
    }
}

__device__ __forceinline__ void load_tile(const uint32_t *ci, int64_t m, int64_t w, uint32_t (&u)[kWQ]) {
    const int64_t e = w * kWE + kWQ * (int64_t)lane_id();
    if (e + kWQ <= m) {
#pragma unroll
        for (int j = 0; j < kWQ / 4; ++j) {
            const uint4 x = __ldcs(reinterpret_cast<const uint4 *>(ci + e) + j);
            u[4 * j] = x.x;
            u[4 * j + 1] = x.y;
            u[4 * j + 2] = x.z;
            u[4 * j + 3] = x.w;
        }
    } else {
#pragma unroll
        for (int q = 0; q < kWQ; ++q) u[q] = e + q < m ? __ldcs(ci + e + q) : 0u;
    }
}

#ifndef GC_CW_PREFETCH
#define GC_CW_PREFETCH 0  // 1: the next warp tile's column ids loaded before the current one is counted (measured: 1.39 vs 1.23 ms
                          // without -- 71 vs 55 registers, 24 vs 32 warps per SM)
#endif
#ifndef GC_CW_MINB
#define GC_CW_MINB 1
#endif
constexpr bool kCwPrefetch = GC_CW_PREFETCH != 0;
__global__ void __launch_bounds__(kWT, GC_CW_MINB) k_count_warp(const int64_t *__restrict__ ro, const uint32_t *__restrict__ ci,
                                                    int64_t n, int64_t m, int64_t nch,
                                                    const uint32_t *__restrict__ crow, uint32_t key,
                                                    unsigned long long *cnt, int jp) {
    __shared__ long long offs_sh[kWT / 32][33];
    __shared__ uint32_t h_sh[kWT / 32][32];
    const unsigned lane = lane_id(), wib = threadIdx.x >> 5;
    long long *offs = offs_sh[wib];
    uint32_t *hs = h_sh[wib];
    hs[lane] = 0u;
    const int64_t nwarps = (int64_t)gridDim.x * (kWT / 32);
    int64_t w = (int64_t)blockIdx.x * (kWT / 32) + wib;
    if (w >= nch) return;
    uint32_t u[kWQ], un[kWQ];
    load_tile(ci, m, w, u);
    for (;;) {
        const int64_t wn = w + nwarps;
        if (kCwPrefetch && wn < nch) load_tile(ci, m, wn, un);  // next tile's column ids in flight
        const int64_t e0 = w * kWE, e1 = min(m, e0 + kWE);
        const int64_t ra = crow[w], rz = crow[w + 1];  // rows touching the tile: [ra, rz]
        const bool last_tile = w == nch - 1;
        const int64_t qf = e0 + kWQ * (int64_t)lane;
        uint32_t mx[kWQ];  // the entries' priorities
#pragma unroll
        for (int q = 0; q < kWQ; ++q) mx[q] = weight_mix(u[q] ^ key);
        int cur = 0;  // this lane's entries < cur are counted
        for (int64_t rb = ra; rb <= rz; rb += 32) {
            int nr = (int)min((int64_t)32, rz - rb + 1);
            offs[lane] = lane <= nr ? (long long)__ldg(ro + rb + lane) : 0ll;
            if (lane == 0) offs[32] = nr == 32 ? (long long)__ldg(ro + rb + 32) : 0ll;
            __syncwarp();
            if (nr == 32 && offs[0] == offs[32] && rb + 32 <= rz) {
                // 32 rows without entries and more to come (a run of isolated
                // vertices): jump to the last empty row before the next row with
                // entries (binary search in the offsets; empty rows are the init
                // phase's), so a long run costs log n, not n / 32, steps
                const long long e = offs[0];
                int64_t lo = rb + 32, hi = rz + 1;  // ro[lo] == e; the first r with ro[r] > e is in (lo, hi]
                if (__ldg(ro + hi) == e) {
                    rb = rz + 1 - 32;  // (no entries up to rz + 1: nothing left in this tile)
                } else {
                    while (hi - lo > 1) {
                        const int64_t mid = lo + ((hi - lo) >> 1);
                        if (__ldg(ro + mid) == e) lo = mid;
                        else hi = mid;
                    }
                    rb = lo - 32;  // ro[lo] == e < ro[lo + 1]: row lo is the next with entries; += 32 lands on it
                }
                __syncwarp();
                continue;
            }
            const int64_t lim = min((int64_t)offs[nr], e1);  // entries of these rows within the tile
            // this lane's entries [cur, qlim) of these rows, one row per step:
            // the row's hi count = popcount of the entries whose priority beats
            // the row vertex's (a 16-bit mask, no per-entry branches)
            const int qlim = (int)max((int64_t)cur, min((int64_t)kWQ, lim - qf));
            bool act = cur < qlim;
            int ri = 0;
            if (act) {
                const int64_t es = qf + cur;
                int lo = 0, hi = nr;  // offs[lo] <= es < offs[hi]
                while (hi - lo > 1) {
                    const int mid = (lo + hi) >> 1;
                    if (offs[mid] <= es) lo = mid;
                    else hi = mid;
                }
                ri = lo;
            }
            int qs = cur;
            while (__any_sync(kFull, act)) {
                if (act) {
                    const int re_rel = (int)min((int64_t)offs[ri + 1] - qf, (int64_t)qlim);  // > qs
                    const uint32_t pv = weight_mix((uint32_t)(rb + ri) ^ key);
                    uint32_t g = 0;
#pragma unroll
                    for (int q = 0; q < kWQ; ++q) g |= (mx[q] > pv ? 1u : 0u) << q;
                    const uint32_t rng = ((1u << re_rel) - 1u) & ~((1u << qs) - 1u);
                    const uint32_t hcount = (uint32_t)__popc(g & rng);
                    if (hcount) atomicAdd(&hs[ri], hcount);
                    qs = re_rel;
                    act = qs < qlim;
                    if (act) {  // the next row with entries here (skip empty rows)
                        do {
                            ++ri;
                        } while (offs[ri + 1] - qf <= qs);
                    }
                }
            }
            cur = qlim;
            __syncwarp();
            if (lane < (unsigned)nr) {
                const int64_t r = rb + lane;
                const int64_t rs = offs[lane], re = offs[lane + 1];
                const uint32_t h = hs[lane];
                hs[lane] = 0u;
                if (rs < e0 || re > e1) {  // crosses a tile boundary: this tile's part
                    const int64_t len = min(re, e1) - max(rs, e0);
                    if (len > 0)
                        atomicAdd(cnt + r, ((unsigned long long)h << 32) + (jp ? 0ull : (unsigned long long)(len - h)));
                } else if (re > rs && (r < rz || last_tile)) {
                    // inside the tile (rows without entries are left to the init phase);
                    // row rz starting at e1 is the next tile's first row
                    cnt[r] = ((unsigned long long)h << 32) | (unsigned long long)(jp ? 1 : (re - rs) - h);
                }
            }
            __syncwarp();
        }
        if (wn >= nch) break;
        w = wn;
        if (kCwPrefetch) {
#pragma unroll
            for (int q = 0; q < kWQ; ++q) u[q] = un[q];
        } else {
            load_tile(ci, m, w, u);
        }
    }
}

template <bool PROF, bool JP, bool MH>
int launch(gc_graph *g, CArgs &a, int *blocks_out) {
    int per_sm = 0;
    GC_CUDA_TRY(cudaFuncSetAttribute(k_count_persistent<PROF, JP, MH>,
                                     cudaFuncAttributeMaxDynamicSharedMemorySize, (int)kStageBytes));
    GC_CUDA_TRY(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k_count_persistent<PROF, JP, MH>,
                                                              threads_for<JP, MH>(), kStageBytes));
    if (per_sm < 1) {
        set_error("persistent count kernel cannot be resident");
        return GC_ERR_CUDA;
    }
    int blocks = per_sm * g->sm_count;
    if (const char *eb = std::getenv("GC_COUNT_BLOCKS")) {  // experiments: fewer / more blocks
        const int b = std::atoi(eb);
        if (b >= 1 && b <= blocks) blocks = b;
    }
    if (blocks >= 2048) {  // the round word's arrival field has 11 bits
        set_error("persistent count kernel: too many blocks for the round word");
        return GC_ERR_CUDA;
    }
    // L2 persistence for the count words (every round's decrements are a
    // burst of random 8-byte atomics; a burst that misses L2 is several times
    // slower, tools/microbench_atomics.cu).  Per-launch attribute: no stream
    // or device state is changed except the persisting-L2 carve-out.
    cudaLaunchAttribute attrs[2];
    int na = 0;
    attrs[na].id = cudaLaunchAttributeCooperative;
    attrs[na].val.cooperative = 1;
    ++na;
    int dev = 0, max_persist = 0, max_window = 0;
    cudaGetDevice(&dev);
    cudaDeviceGetAttribute(&max_persist, cudaDevAttrMaxPersistingL2CacheSize, dev);
    cudaDeviceGetAttribute(&max_window, cudaDevAttrMaxAccessPolicyWindowSize, dev);
    const char *env = std::getenv("GC_L2_PERSIST");
    // opt-in only: measured slower on R-MAT s24 (40.6 vs 35.7 ms)
    const bool persist = max_persist > 0 && max_window > 0 && env && env[0] == '1';
    if (persist) {
        size_t cur = 0;
        cudaDeviceGetLimit(&cur, cudaLimitPersistingL2CacheSize);
        if (cur < (size_t)max_persist) cudaDeviceSetLimit(cudaLimitPersistingL2CacheSize, (size_t)max_persist);
        const bool pk = GC_PACKED && !JP && !MH;  // the rounds' count words: 32-bit packed or 64-bit
        const size_t bytes = std::min<size_t>((size_t)a.n * (pk ? 4 : 8), (size_t)max_window);
        attrs[na].id = cudaLaunchAttributeAccessPolicyWindow;
        attrs[na].val.accessPolicyWindow.base_ptr = pk ? (void *)a.cnt32 : (void *)a.cnt;
        attrs[na].val.accessPolicyWindow.num_bytes = bytes;
        attrs[na].val.accessPolicyWindow.hitRatio =
            (float)std::min(1.0, (double)max_persist / (double)std::max<size_t>(bytes, 1));
        attrs[na].val.accessPolicyWindow.hitProp = cudaAccessPropertyPersisting;
        attrs[na].val.accessPolicyWindow.missProp = cudaAccessPropertyStreaming;
        ++na;
    }
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3(blocks);
    cfg.blockDim = dim3(threads_for<JP, MH>());
    cfg.dynamicSmemBytes = kStageBytes;
    cfg.stream = g->stream;
    cfg.attrs = attrs;
    cfg.numAttrs = na;
    GC_CUDA_TRY(cudaLaunchKernelEx(&cfg, k_count_persistent<PROF, JP, MH>, a));
    *blocks_out = blocks;
    return GC_OK;
}

}  // namespace

// Scratch of COUNT mode (allocated on first use, kept with the handle).
namespace {
// vertices of degree > dmin (big: > kPackMax; JP slots: > kShortMax),
// counted, at most cap of them recorded
__global__ void k_find_big(const int64_t *__restrict__ ro, int64_t n, int64_t dmin, uint32_t *big,
                           int cap, unsigned long long *nbig) {
    for (int64_t v = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; v < n;
         v += (int64_t)gridDim.x * blockDim.x) {
        if (ro[v + 1] - ro[v] > dmin) {
            const unsigned long long i = atomicAdd(nbig, 1ull);
            if (i < (unsigned long long)cap) big[i] = (uint32_t)v;
        }
    }
}

// number of vertices of degree > dmin
int count_deg_above(gc_graph *g, int64_t dmin, uint32_t *big, int cap, unsigned long long *out) {
    unsigned long long *d = nullptr;
    GC_CUDA_TRY(dmalloc(&d, 8));
    GC_CUDA_TRY(cudaMemsetAsync(d, 0, 8, g->stream));
    if (g->n > 0)
        k_find_big<<<g->sm_count * 4, 256, 0, g->stream>>>(g->ro, g->n, dmin, big, cap, d);
    GC_CUDA_TRY(cudaMemcpyAsync(out, d, 8, cudaMemcpyDeviceToHost, g->stream));
    GC_CUDA_TRY(cudaStreamSynchronize(g->stream));
    dfree(d);
    return GC_OK;
}
}  // namespace

int ensure_count_scratch(gc_graph *g) {
    Scratch &s = g->s;
    const size_t nn = (size_t)std::max<int64_t>(g->n, 1);
    if (s.cnt) return GC_OK;
    // big vertices: seed-independent, found once per graph
    GC_CUDA_TRY(dmalloc(&s.big, (size_t)(kHTab / 2) * 4));
    GC_CUDA_TRY(dmalloc(&s.big32, (size_t)(3 * kHTab) * 4));
    GC_CUDA_TRY(dmalloc(&s.cnt32, nn * 4));
    {
        unsigned long long h = 0;
        int rc = count_deg_above(g, kPackMax, s.big, kHTab / 2, &h);
        if (rc) return rc;
        s.nbig = h <= (unsigned long long)(kHTab / 2) ? (int)h : -1;  // -1: too many to pack
    }
    GC_CUDA_TRY(dmalloc(&s.cnt, nn * 8));
    GC_CUDA_TRY(dmalloc(&s.Z, nn * 4));
    s.sl_cap = (int64_t)nn;
    s.wl_cap = (int64_t)nn + g->nnz / kSeg + 1;
    // one monotone array per barrier group (each could receive every item)
    GC_CUDA_TRY(dmalloc(&s.SL, (size_t)kNG * (size_t)s.sl_cap * sizeof(Item)));
    GC_CUDA_TRY(dmalloc(&s.WL, (size_t)kNG * (size_t)s.wl_cap * sizeof(Item)));
    // (recycled memory could hold tagged items of another handle's colouring)
    GC_CUDA_TRY(cudaMemsetAsync(s.SL, 0, (size_t)kNG * (size_t)s.sl_cap * sizeof(Item), g->stream));
    GC_CUDA_TRY(cudaMemsetAsync(s.WL, 0, (size_t)kNG * (size_t)s.wl_cap * sizeof(Item), g->stream));
    s.count_epoch = 0;
    // hub chunk list: at most nnz / kHubChunk entries
    GC_CUDA_TRY(dmalloc(&s.hubs, ((size_t)g->nnz / kHubChunk + 1) * 8));
    GC_CUDA_TRY(dmalloc(&s.cctr, kCCtrWords * sizeof(unsigned long long)));
    GC_CUDA_TRY(dmalloc(&s.cM, (nn + 31) / 32 * 4));
    return GC_OK;
}

// tiled counting pass: the row of every tile's first entry, for the CSR the
// handle colours now (a deduplicated copy replaces it at most once)
static int ensure_crow(gc_graph *g) {
    Scratch &s = g->s;
    if (s.crow && s.crow_ro == g->ro && s.crow_nnz == g->nnz) return GC_OK;
    dfree(s.crow);
    s.crow = nullptr;
    s.nch = std::max<int64_t>(1, (g->nnz + kTE - 1) / kTE);
    GC_CUDA_TRY(dmalloc(&s.crow, (size_t)(s.nch + 1) * 4));
    k_chunk_rows<<<g->sm_count * 4, 256, 0, g->stream>>>(g->ro, g->n, s.nch, s.crow);
    GC_CUDA_TRY(cudaGetLastError());
    s.crow_ro = g->ro;
    s.crow_nnz = g->nnz;
    return GC_OK;
}

__global__ void k_degrees(const int64_t *__restrict__ ro, int64_t n, uint32_t *deg) {
    for (int64_t v = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; v < n; v += (int64_t)gridDim.x * blockDim.x)
        deg[v] = (uint32_t)min(ro[v + 1] - ro[v], (int64_t)0xFFFFFFFF);
}

// LDF: deg[v] = row length (rows are strictly increasing here: gc_api runs
// ensure_strict_rows first, so it is the number of distinct neighbours)
static int ensure_degrees(gc_graph *g) {
    Scratch &s = g->s;
    if (s.deg) return GC_OK;
    GC_CUDA_TRY(dmalloc(&s.deg, (size_t)std::max<int64_t>(g->n, 1) * 4));
    if (g->n > 0) k_degrees<<<g->sm_count * 8, 256, 0, g->stream>>>(g->ro, g->n, s.deg);
    GC_CUDA_TRY(cudaGetLastError());
    return GC_OK;
}

// JP mex slots: one per vertex of degree > kShortMax (each is scheduled once)
static int ensure_jp_scratch(gc_graph *g) {
    Scratch &s = g->s;
    if (s.jslot) return GC_OK;
    unsigned long long h = 0;
    int rc = count_deg_above(g, kShortMax, nullptr, 0, &h);
    if (rc) return rc;
    s.jslot_cap = (int64_t)h;
    GC_CUDA_TRY(dmalloc(&s.jslot, ((size_t)h + 1) * kSlotWords * 4));
    return GC_OK;
}

static int run_count(gc_graph *g, const RunParams &p, RunResult *r, int jpv) {
    NvtxRange nv_(jpv ? "COUNT colouring (JP)" : p.H > 1 ? "COUNT colouring (multi-hash)" : "COUNT colouring (max-min)");
    Scratch &s = g->s;
    const int64_t n = g->n;
    const bool jp = jpv != 0;
    const bool mh = !jp && p.H > 1;
    r->rounds = r->inner = r->launches = 0;
    r->max_color = -1;  // (set only by a run that completes)
    if (n == 0) return GC_OK;
    if (n >= (1ll << 29)) {  // a round's SL items could pass the round word's 29-bit field
        set_error("COUNT mode: n >= 2^29 exceeds the round word's item field");
        return GC_ERR_TOO_LARGE;
    }
    int rc = ensure_count_scratch(g);
    if (rc) return rc;
    if (mh && s.cnt_h < p.H) {  // H count words per vertex
        dfree(s.cnt);
        s.cnt = nullptr;
        GC_CUDA_TRY(dmalloc(&s.cnt, (size_t)n * 8 * (size_t)p.H));
        s.cnt_h = p.H;
    }
    if (jpv == 1 && (rc = ensure_jp_scratch(g))) return rc;
    if (GC_PACKED && s.nbig < 0) {  // more big vertices than the shared hash set holds
        if (jp) return run_luby(g, p, r);
        if (mh) return run_sweep_maxmin(g, p, r);
        rc = ensure_scratch(g, true, false);
        return rc ? rc : run_persistent_maxmin(g, p, r);
    }
    // max-min colours >= 2 vertices of every uncoloured component per round;
    // JP >= 1 (its rounds are the longest decreasing-weight path)
    const int64_t max_rounds = std::min<int64_t>(std::min<int64_t>(p.max_rounds, 0xFFFFFFF0ll),
                                                 jp ? n + 2 : mh ? std::min<int64_t>(n / 2 + 2, (1ll << 27) - 2)
                                                             : n / 2 + 2);
    rc = ensure_nk(g, std::min<int64_t>(std::min<int64_t>(n + 2, max_rounds + 2), 1 << 20));
    if (rc) return rc;
    cudaStream_t st = g->stream;
    GC_CUDA_TRY(cudaMemsetAsync(s.cctr, 0, kCCtrWords * sizeof(unsigned long long), st));
    const bool prof = p.prof && p.prof->on;
    // the counting pass and the persistent kernel are bracketed by events on
    // every colouring (un-instrumented kernels: gc_stats kernel_ms[1] / [0])
    EventPair ev01;
    cudaEvent_t e0 = nullptr, e1 = nullptr, e2 = nullptr;
    GC_CUDA_TRY(cudaEventCreate(&ev01.e0));
    GC_CUDA_TRY(cudaEventCreate(&ev01.e1));
    e0 = ev01.e0;
    e1 = ev01.e1;
    EventPair ev2;
    GC_CUDA_TRY(cudaEventCreate(&ev2.e0));
    e2 = ev2.e0;
    GC_CUDA_TRY(cudaEventRecord(e0, st));
    const uint32_t key = p.keys.k[0];
    unsigned long long *nhubs = s.cctr + cHubs;
    // LDF: the degree array, built once per graph (seed-independent)
    const uint32_t *dg = nullptr;
    if (p.ldf) {
        if ((rc = ensure_degrees(g))) return rc;
        dg = s.deg;
    }
    {
        const int64_t warps = (n + 31) / 32;
        const int blocks = (int)std::min<int64_t>((warps + 7) / 8, (int64_t)g->sm_count * 16);
        uint2 *hubs = reinterpret_cast<uint2 *>(s.hubs);
        CountKeys ck;
        ck.H = p.H;
        for (int j = 0; j < GC_MAX_HASHES; ++j) ck.k[j] = p.keys.k[j];
        if (mh) {
            k_count<true><<<blocks, 256, 0, st>>>(g->ro, g->ci, n, ck, s.cnt, hubs, nhubs, 0, nullptr);
            k_count_hub<true><<<g->sm_count * 8, 256, 0, st>>>(g->ro, g->ci, ck, s.cnt, hubs, nhubs, 0,
                                                               nullptr);
        } else if (kCountStream && !dg && ((reinterpret_cast<uintptr_t>(g->ci) | reinterpret_cast<uintptr_t>(g->ro)) & 15) == 0) {
            // (cp.async copies 16-byte pieces: borrowed buffers must be 16-byte aligned)
            if ((rc = ensure_crow(g))) return rc;
            const int64_t nch = s.nch;
            k_count_zero<<<g->sm_count, 256, 0, st>>>(g->ro, s.crow, nch, s.cnt, jp ? 1 : 0);
            k_count_warp<<<(int)std::min<int64_t>((nch + 7) / 8, (int64_t)g->sm_count * 8), kWT, 0, st>>>(
                g->ro, g->ci, n, g->nnz, nch, s.crow, key, s.cnt, jp ? 1 : 0);
        } else {
            k_count<false><<<blocks, 256, 0, st>>>(g->ro, g->ci, n, ck, s.cnt, hubs, nhubs, jp ? 1 : 0, dg);
            k_count_hub<false><<<g->sm_count * 8, 256, 0, st>>>(g->ro, g->ci, ck, s.cnt, hubs, nhubs,
                                                                jp ? 1 : 0, dg);
        }
        GC_CUDA_TRY(cudaGetLastError());
    }
    GC_CUDA_TRY(cudaEventRecord(e1, st));
    CArgs a;
    a.ro = g->ro;
    a.ci = g->ci;
    a.C = s.C;
    a.cnt = s.cnt;
    a.cnt32 = s.cnt32;
    a.big32 = s.big32;
    a.big = s.big;
    a.nbig = std::max(s.nbig, 0);
    a.Zlo = s.Z;
    a.SL = reinterpret_cast<Item *>(s.SL);
    a.WL = reinterpret_cast<Item *>(s.WL);
    a.ctr = s.cctr;
    a.nk = s.nk;
    a.rstat = s.rstat;
    a.nk_cap = s.nk_cap;
    a.n = n;
    a.key = key;
    a.max_rounds = (uint32_t)max_rounds;
    if (const char *e = std::getenv("GC_MAX_ROUNDS"))  // (experiments: stop after a few rounds)
        a.max_rounds = (uint32_t)std::min<int64_t>(max_rounds, std::max(0, std::atoi(e)));
    a.sl_cap = (unsigned long long)s.sl_cap;
    a.wl_cap = (unsigned long long)s.wl_cap;
    a.jslot = s.jslot;
    a.jslot_cap = (unsigned long long)s.jslot_cap;
    a.H = p.H;
    for (int j = 0; j < GC_MAX_HASHES; ++j) a.mkeys[j] = p.keys.k[j];
    a.dg = dg;
    // item round tags (merged hand-off): a new epoch per colouring; the item
    // arrays are cleared when the 8-bit epoch wraps (a stale item then
    // cannot carry a current tag); epoch 0 (the cleared state) is never used
    if (++s.count_epoch % 256u == 0u) {
        GC_CUDA_TRY(cudaMemsetAsync(s.SL, 0, (size_t)kNG * (size_t)s.sl_cap * sizeof(Item), st));
        GC_CUDA_TRY(cudaMemsetAsync(s.WL, 0, (size_t)kNG * (size_t)s.wl_cap * sizeof(Item), st));
        ++s.count_epoch;
    }
    a.epoch = s.count_epoch;
    // JP rounds relaxed for Luby and Alg.2 (Alg.4's per-round colour sets stay
    // behind release / acquire barriers); Luby's mex slots zeroed up front
    a.jrel = (jp && jpv != 3 && kRelaxedArrive && !std::getenv("GC_JP_NO_RELAX")) ? 1 : 0;
    if (a.jrel && jpv == 1 && s.jslot)
        GC_CUDA_TRY(cudaMemsetAsync(s.jslot, 0, ((size_t)s.jslot_cap + 1) * kSlotWords * 4, st));
    a.M = s.cM;
    a.jpv = jpv;
    a.cr = nullptr;
    a.B = nullptr;
    a.bwords = 0;
    if (jpv == 3) {  // Alg.4: per-round colours + 3 colour sets (colours <= rounds)
        const int64_t words = (max_rounds + 64) / 32;
        if (!s.jcr || s.jcr_words < words) {
            dfree(s.jcr);
            s.jcr = nullptr;
            GC_CUDA_TRY(dmalloc(&s.jcr, (size_t)(max_rounds + 2 + 3 * words) * 4));
            s.jcr_words = words;
        }
        a.cr = s.jcr;
        a.B = s.jcr + max_rounds + 2;
        a.bwords = (uint32_t)words;
        GC_CUDA_TRY(cudaMemsetAsync(a.B, 0, (size_t)3 * words * 4, st));
    }
    if (prof) GC_CUDA_TRY(cudaMemsetAsync(s.rstat, 0, sizeof(int64_t) * 16 * (size_t)s.nk_cap, st));
    int blocks = 0;
    if (jp) rc = prof ? launch<true, true, false>(g, a, &blocks) : launch<false, true, false>(g, a, &blocks);
    else if (mh) rc = prof ? launch<true, false, true>(g, a, &blocks) : launch<false, false, true>(g, a, &blocks);
    else rc = prof ? launch<true, false, false>(g, a, &blocks) : launch<false, false, false>(g, a, &blocks);
    if (rc) return rc;
    r->launches += 3;  // k_count, k_count_hub, persistent kernel
    GC_CUDA_TRY(cudaEventRecord(e2, st));
    unsigned long long h[kCCtrWords];
    GC_CUDA_TRY(cudaMemcpyAsync(h, s.cctr, sizeof(h), cudaMemcpyDeviceToHost, st));
    GC_CUDA_TRY(cudaStreamSynchronize(st));
    if (h[cErr] != 0) {
        char buf[200];
        if (h[cErr] == 4 || h[cErr] == 5 || h[cErr] == 7)
            snprintf(buf, sizeof(buf), "count underflow at vertex %llu in round %llu: the adjacency is "
                     "not symmetric", h[cErr + 2], h[cErr + 1]);
        else
            snprintf(buf, sizeof(buf), "internal consistency check %llu failed in round %llu (vertex %llu)",
                     h[cErr], h[cErr + 1], h[cErr + 2]);
        if (h[cErr] == 9) {  // one round reserved more items than the round word's fields hold
            set_error("COUNT mode: a round's items overflowed the round word (2^29 short / 2^24 long items)");
            return GC_ERR_TOO_LARGE;
        }
        set_error(buf);
        return (h[cErr] == 4 || h[cErr] == 5 || h[cErr] == 7) ? GC_ERR_NOT_SYMMETRIC : GC_ERR_CUDA;
    }
    if (h[cCol] != (unsigned long long)n) {
        set_error("count-mode colouring stalled with uncoloured vertices: the adjacency is not symmetric");
        return GC_ERR_NOT_SYMMETRIC;
    }
    r->rounds = (int64_t)h[cRounds];
    r->max_color = h[cMaxC] ? (int64_t)h[cMaxC] - 1 : -1;  // (relaxed rounds' final pass)
    r->inner = r->rounds;
    if (p.prof) {
        // class 0: the persistent kernel; 1: counting kernels (both timed on
        // every colouring); PROF only: 2 its init phase (round 0), 3 its
        // rounds (globaltimer, block 0), algorithmic bytes
        float ms_all = 0.f, ms_cnt = 0.f;
        cudaEventElapsedTime(&ms_all, e0, e2);
        cudaEventElapsedTime(&ms_cnt, e0, e1);
        p.prof->ms[0] += ms_all - ms_cnt;
        p.prof->launches[0] += 1;
        p.prof->launch_us.push_back(1e3f * (ms_all - ms_cnt));
        p.prof->ms[1] += ms_cnt;
        p.prof->launches[1] += 2;
        if (!prof) p.prof->visits += (int64_t)h[cVis];  // count decrements issued (always counted)
    }
    if (prof) {
        p.prof->ms[2] += (double)h[cPhaseNs] / 1e6;
        p.prof->ms[3] += (double)h[cPhaseNs + 1] / 1e6;
        // algorithmic bytes.  Counting: 8 B offsets + 8 B
        // count per vertex + 4 B per entry.  Persistent kernel: init 8 B
        // count + 8 B Z + 4 B colour + 8 B offsets (coloured in round 0) per
        // vertex + n/8 B schedule bits; per scheduled vertex 16 B item write
        // + 16 B item read + 8 B offsets + 8 B Z + 4 B colour; per walked
        // entry 4 B column id + 8 B count read + 8 B count write.
        const int64_t vis = (int64_t)h[cVis];
        const int64_t m = g->nnz;
        p.prof->bytes[1] += 16 * n + 4 * m;
        p.prof->bytes[0] += 28 * n + n / 8 + 52 * n + 20 * vis;
        p.prof->visits += vis;
    }
    return GC_OK;
}

int run_count_maxmin(gc_graph *g, const RunParams &p, RunResult *r) { return run_count(g, p, r, 0); }
int run_count_jp(gc_graph *g, const RunParams &p, RunResult *r, int jpv) { return run_count(g, p, r, jpv); }

}  // namespace gc
