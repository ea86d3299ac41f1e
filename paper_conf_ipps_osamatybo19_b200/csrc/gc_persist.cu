// gc_persist.cu -- EVENT mode as ONE persistent cooperative kernel that runs
// every round of the max-min colouring (Alg.1 + Alg.5, P:L102-113,
// P:L506-556; H = 1), one grid barrier per round.
//
// The method per round is the witness/resume scheme of gc_event.cu (see its
// header and DESIGN.md 7.1); this file only schedules it on the 148 SMs.
//
// Round 0 (every vertex evaluated) runs as three phases over static lists:
//   R0a lane per vertex, 8-entry window (kLaneWin); unresolved rows -> WQ0;
//   R0b WQ0: warp per vertex, 256-entry window (kWarpWin); longer -> long scan;
//   R0c long scans split into kSeg-entry segments over all warps.
// Every later round k is ONE phase M_k driven by a dynamic work queue:
//   - it starts with the NOTIFY items of the vertices coloured in round k-1
//     (appended during M_{k-1}: short rows as one item, long rows as
//     kNotifySeg-entry segments);
//   - a NOTIFY item wakes the uncoloured neighbours that used the coloured
//     vertex as a witness (dedupe: atomicMax round stamp) and pushes EVAL(k)
//     items into the same queue;
//   - EVAL(k) evaluates one vertex with a warp (256-entry window), pushing
//     SCAN(k) segment items for longer rows into the same queue;
//   - a vertex coloured in round k pushes its NOTIFY items into the NEXT
//     round's queue.
// This is exact: round-k evaluation needs the colours of rounds < k (all
// written during earlier phases) and counts colours written concurrently in
// round k as uncoloured (C[u] >= 2k), i.e. the snapshot of Alg.5 L26 (R6).  A
// NOTIFY(k-1) item may race with the evaluation of the neighbour it targets:
// the stamp makes the wake unique, and a witness chosen in round k that is
// itself coloured in round k wakes the vertex through NOTIFY(k) in M_{k+1}.
// The phase ends when the queue is drained: done == tail, read in that order
// (tail is monotone and a producer appends before it completes its own item).
#include <cstdio>
#include <vector>

#include "gc_event_common.cuh"

namespace gc {

int fill_u32(uint32_t *p, uint32_t val, int64_t n, cudaStream_t st);
int ensure_nk(gc_graph *g, int64_t need);

namespace {

using namespace ev;

constexpr int kThreads = 512;
constexpr int kLaneWin = 8;      // entries a lane scans in round 0 before handing off
constexpr int kWarpWin = 256;    // entries a warp scans before splitting
constexpr int kSeg = 256;        // entries per long-scan segment (8 per lane)
constexpr int kNotifySeg = 128;  // entries per notify segment (4 per lane)
constexpr int kLaneNotify = 32;  // rows up to this length are one notify item
constexpr unsigned long long kDynWarps = 2048;  // warps that serve the dynamic queue

// work items: {a, (type << 28) | b}; type 0 marks an empty slot
enum : uint32_t { T_NOTIFY = 1u, T_EVAL = 2u, T_SCAN = 3u };
constexpr uint32_t kSub = 0x0FFFFFFFu;

// ctr layout
enum : int {
    r0WQ = 0, r0SQ = 1, r0LS = 2,  // static rounds 0 and 1: lists (3 slots per round)
    r0B = 6,                       // vertices left blocked by round 0 (list B0)
    kQ = 24,                       // two queue sets of 8 (by round parity)
    kRem = 40,
    kVisE = 41,
    kVisS = 42,
    kVisN = 43,
    kSumD = 44,
    kRounds = 45,
    kColTotal = 46,                // vertices coloured so far
    kPhaseNs = 50,                 // [50..53] PROF
    kErr = 56,                     // [56..58] first trap (kind, round, vertex)
    kErrPar = 59,                  // [59..60] a trap fired in a round of this parity
    kBar = 61,                     // [61..62] grid barrier count / generation
    kAbort = 63
};
enum : int { qTail = 0, qHead = 1, qDone = 2, qLS = 3, qEval = 4 };

struct LongScan {   // one slot per long scan of a round (32 B)
    uint32_t v;
    uint32_t ticket;  // segments still outstanding
    uint32_t minH;    // first hi hit, relative to the row start (kNone: none)
    uint32_t minL;
    uint32_t need;    // bit 0: hi still searched, bit 1: lo
    uint32_t sh, sl;  // search starts (relative)
    uint32_t base;    // relative start of segment 0
};

struct Args {
    const int64_t *ro;
    const uint32_t *ci;
    uint32_t *C;
    uint2 *W;
    uint2 *P;
    uint32_t *S;
    uint32_t *WQ0;   // static rounds: unresolved lane windows
    uint2 *SQ0;      // static rounds: long-scan segments
    uint32_t *B0;    // vertices left blocked by round 0 (round 1 re-checks them)
    LongScan *LS;
    uint2 *Q[2];     // work queues by round parity
    unsigned long long *qc;  // queue counters: set s, counter c at qc[(8 s + c) * 16]
    unsigned long long *ctr;
    int64_t *nk;
    int64_t *rstat;
    int64_t nk_cap;
    int64_t n;
    uint32_t key;
    uint32_t max_rounds;
    unsigned long long q_cap, sq_cap, ls_cap;
    unsigned long long dyn_warps;  // warps serving the dynamic queue
    uint32_t *owner;               // debug: slot owner (round << 1 | busy)
    int split;                     // debug: NOTIFY items in a static sub-phase first
};

// Queue counters live on separate 128-byte lines: idle warps poll qDone/qTail
// while busy warps update them, and a shared line would serialise both.
__device__ __forceinline__ unsigned long long *QC(const Args &a, int set, int c) {
    return a.qc + (8 * set + c) * 16;
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

// Internal-consistency trap: record the first violation (kind, round, vertex)
// instead of writing out of bounds; ctr[kErrPar + (k & 1)] makes the whole
// grid leave at the next barrier.
__device__ __forceinline__ void flag_error(const Args &a, unsigned kind, uint32_t k, uint32_t v) {
    if (atomicCAS(&a.ctr[kErr], 0ull, (unsigned long long)kind) == 0ull) {
        a.ctr[kErr + 1] = k;
        a.ctr[kErr + 2] = v;
    }
    a.ctr[kErrPar + (k & 1)] = 1;
}

// Grid-wide barrier (cooperative launch: all blocks resident).  Generation
// barrier on ctr[kBar..kBar+1]; the last block to arrive resets the count,
// zeroes the queue set `reset_set` (the set the next phase appends NOTIFY
// items to; its previous use is over), then bumps the generation.  A wait
// longer than kBarrierTimeoutNs records a trap and makes every block leave
// (returns false) instead of hanging.  Each thread then issues a gpu-scope
// fence: the next phase reads state other SMs wrote, and L1 is not coherent.
constexpr unsigned long long kBarrierTimeoutNs = 4000000000ull;

__device__ __forceinline__ bool grid_barrier(const Args &a, int id, uint32_t k, int reset_set) {
    __shared__ int ok_sh;
    __syncthreads();
    if (threadIdx.x == 0) {
        int ok = 1;
        volatile unsigned long long *gen = a.ctr + kBar + 1;
        volatile unsigned long long *abort = a.ctr + kAbort;
        const unsigned long long g0 = *gen;
        __threadfence();
        const unsigned long long arrived = atomicAdd(a.ctr + kBar, 1ull) + 1;
        if (arrived == gridDim.x) {
            a.ctr[kBar] = 0;
            if (reset_set >= 0)
                for (int i = 0; i < 8; ++i) *QC(a, reset_set, i) = 0;
            __threadfence();
            atomicAdd(a.ctr + kBar + 1, 1ull);
        } else {
            const unsigned long long t0 = gtimer();
            while (*gen == g0) {
                if (*abort) {
                    ok = 0;
                    break;
                }
                if (gtimer() - t0 > kBarrierTimeoutNs) {
                    flag_error(a, 100 + id, k, blockIdx.x);
                    atomicExch(a.ctr + kAbort, 1ull);
                    ok = 0;
                    break;
                }
                __nanosleep(32);
            }
        }
        __threadfence();
        ok_sh = ok;
    }
    __syncthreads();
    __threadfence();
    return ok_sh != 0;
}

// Publish one item at slot `pos` of queue q: payload first, type tag last.
__device__ __forceinline__ void put_item(const Args &a, int q, unsigned long long pos, uint2 it,
                                         uint32_t k) {
    if (pos >= a.q_cap) {
        flag_error(a, 1, k, it.x);
        return;
    }
    volatile uint2 *dst = reinterpret_cast<volatile uint2 *>(&a.Q[q][pos]);
    dst->x = it.x;
    __threadfence();
    dst->y = it.y;
}

// Append `cnt` items generated by `make(i)` (whole warp) to queue q.
template <class Make>
__device__ __forceinline__ void push_items(const Args &a, int q, uint32_t cnt, uint32_t k,
                                           Make make) {
    if (cnt == 0) return;
    unsigned long long b = 0;
    if (lane_id() == 0) b = atomicAdd(QC(a, q, qTail), (unsigned long long)cnt);
    b = __shfl_sync(kFull, b, 0);
    for (uint32_t i = lane_id(); i < cnt; i += 32) put_item(a, q, b + i, make(i), k);
}

// After a settle in round k (whole warp converged): count the coloured lanes
// and queue their NOTIFY items for round k+1.  Round 0 records the vertices it
// leaves blocked instead: round 1 re-checks all of them (cheaper than walking
// the rows of the ~70% of vertices round 0 colours), so round 0 queues no
// NOTIFY items.
__device__ __forceinline__ void colored_notify(const Args &a, bool colored, uint32_t u,
                                               int64_t deg, uint32_t k, bool blocked = false) {
    const int q = (k + 1) & 1;
    if (k == 0) warp_append(blocked, u, a.B0, &a.ctr[r0B]);
    const unsigned m = __ballot_sync(kFull, colored);
    if (!m) return;
    if (lane_id() == (unsigned)(__ffs(m) - 1))
        atomicAdd(&a.ctr[kColTotal], (unsigned long long)__popc(m));
    if (k == 0) return;
    // short rows: one item per vertex, one append per warp
    const bool shortrow = colored && deg <= kLaneNotify;
    const unsigned sm = __ballot_sync(kFull, shortrow);
    if (sm) {
        unsigned long long b = 0;
        const unsigned leader = __ffs(sm) - 1;
        if (lane_id() == leader)
            b = atomicAdd(QC(a, q, qTail), (unsigned long long)__popc(sm));
        b = __shfl_sync(kFull, b, leader);
        if (shortrow)
            put_item(a, q, b + __popc(sm & ((1u << lane_id()) - 1u)),
                     make_uint2(u, (T_NOTIFY << 28) | kSub), k);  // kSub: whole row
    }
    unsigned lm = __ballot_sync(kFull, colored && !shortrow);
    while (lm) {  // long rows: kNotifySeg-entry segments, the whole warp writes
        const int src = __ffs(lm) - 1;
        lm &= lm - 1;
        const uint32_t uu = __shfl_sync(kFull, u, src);
        const int64_t dg = __shfl_sync(kFull, deg, src);
        const uint32_t nseg = (uint32_t)((dg + kNotifySeg - 1) / kNotifySeg);
        push_items(a, q, nseg, k,
                   [&](uint32_t i) { return make_uint2(uu, (T_NOTIFY << 28) | i); });
    }
}

// Lane-serial search of a short window [s, lim) (lim - s <= WIN): all column
// indices first, then all colours, then the in-order first-hit test.
template <int WIN>
__device__ __forceinline__ void lane_window(const Args &a, uint32_t thresh, uint32_t pv,
                                            const Resume &r, int64_t s, int64_t lim, Found &f) {
    uint32_t u[WIN], c[WIN];
#pragma unroll
    for (int q = 0; q < WIN; ++q) u[q] = s + q < lim ? a.ci[s + q] : 0u;
#pragma unroll
    for (int q = 0; q < WIN; ++q) c[q] = s + q < lim ? __ldcg(&a.C[u[q]]) : 0u;
#pragma unroll
    for (int q = 0; q < WIN; ++q) {
        const int64_t e = s + q;
        if (e < lim && c[q] >= thresh) {
            const uint32_t pu = weight_mix(u[q] ^ a.key);
            if (r.need_hi && f.hpos < 0 && e >= r.sh && pu > pv) {
                f.hpos = e;
                f.hw = u[q];
            }
            if (r.need_lo && f.lpos < 0 && e >= r.sl && pu < pv) {
                f.lpos = e;
                f.lw = u[q];
            }
        }
    }
}

// Whole-warp evaluation of one vertex in round k: scan a kWarpWin window;
// resolved -> settle; otherwise open a long scan whose segments go to the
// round-0 list (round 0) or to this round's queue.
template <bool PROF>
__device__ __forceinline__ void eval_warp(const Args &a, uint32_t v, uint32_t k, uint32_t &nvis) {
    const bool dense = k == 0;             // round 0: no witnesses yet
    const bool stat = k <= 1;              // static rounds use the SQ0 list
    const uint32_t thresh = 2u * k;
    const unsigned lane = lane_id();
    const int64_t rs = a.ro[v], re = a.ro[v + 1];
    const Resume r = resume_of(v, rs, dense, a.W, a.P, a.C, thresh);
    if (!r.need_hi && !r.need_lo) return;
    int64_t s = r.need_hi ? r.sh : re;
    if (r.need_lo && r.sl < s) s = r.sl;
    const int64_t lim = min(re, s + (int64_t)kWarpWin);
    Found f;
    uint32_t vis = 0;
    warp_search(a.ci, a.C, thresh, a.key, weight_mix(v ^ a.key), r.need_hi, r.need_lo, r.sh, r.sl,
                lim, f, vis);
    if (PROF) nvis += vis;
    if (lane == 0 && f.hpos >= 0 && (f.hpos < s || f.hpos >= lim)) flag_error(a, 50, k, v);
    if (lane == 0 && f.lpos >= 0 && (f.lpos < s || f.lpos >= lim)) flag_error(a, 51, k, v);
    const bool miss_hi = r.need_hi && f.hpos < 0;
    const bool miss_lo = r.need_lo && f.lpos < 0;
    if (lim < re && (miss_hi || miss_lo)) {
        const uint32_t nseg = (uint32_t)((re - lim + kSeg - 1) / kSeg);
        unsigned long long *lsc = stat ? &a.ctr[r0LS + 3 * k] : QC(a, k & 1, qLS);
        unsigned long long slot = 0;
        if (lane == 0) {
            slot = atomicAdd(lsc, 1ull);
            if (slot < a.ls_cap) {
                const uint32_t prev = atomicExch(&a.owner[slot], (k << 1) | 1u);
                if (prev & 1u) {  // still busy: same round (60) or an earlier one (61)
                    flag_error(a, (prev >> 1) == k ? 60 : 61, k, (uint32_t)slot);
                    a.ctr[47] = prev >> 1;
                }
            }
            if (slot >= a.ls_cap) {
                flag_error(a, 2, k, v);
                slot = ~0ull;
            } else {
                LongScan L;
                L.v = v;
                L.ticket = nseg;
                L.minH = f.hpos >= 0 ? (uint32_t)(f.hpos - rs) : kNone;
                L.minL = f.lpos >= 0 ? (uint32_t)(f.lpos - rs) : kNone;
                L.need = (miss_hi ? 1u : 0u) | (miss_lo ? 2u : 0u) | (k << 2);  // + round tag
                L.sh = (uint32_t)(r.sh - rs);
                L.sl = (uint32_t)(r.sl - rs);
                L.base = (uint32_t)(lim - rs);
                if ((L.minH != kNone && L.minH >= (uint32_t)(re - rs)) ||
                    (L.minL != kNone && L.minL >= (uint32_t)(re - rs)))
                    flag_error(a, 52, k, v);
                a.LS[slot] = L;
                __threadfence();
                if (__ldcg(&a.LS[slot].minL) != L.minL || __ldcg(&a.LS[slot].v) != v)
                    flag_error(a, 53, k, v);
            }
        }
        // every lane publishes SCAN items that point at the slot lane 0 just
        // wrote: __syncwarp orders that store before the lanes' own (fenced)
        // item stores, so a consumer that sees an item sees the slot
        __syncwarp();
        slot = __shfl_sync(kFull, slot, 0);
        if (slot == ~0ull) return;
        if (stat) {
            unsigned long long b = 0;
            if (lane == 0) b = atomicAdd(&a.ctr[r0SQ + 3 * k], (unsigned long long)nseg);
            b = __shfl_sync(kFull, b, 0);
            if (b + nseg > a.sq_cap) {
                if (lane == 0) flag_error(a, 2, k, v);
                return;
            }
            for (uint32_t i = lane; i < nseg; i += 32) a.SQ0[b + i] = make_uint2((uint32_t)slot, i);
        } else {
            // lane 0 wrote the slot, so lane 0 publishes its items: the slot
            // store is then ordered before every item by lane 0's own fences
            if (lane == 0) {
                const unsigned long long b = atomicAdd(QC(a, k & 1, qTail), (unsigned long long)nseg);
                for (uint32_t i = 0; i < nseg; ++i)
                    put_item(a, k & 1, b + i, make_uint2((uint32_t)slot, (T_SCAN << 28) | i), k);
            }
        }
        return;
    }
    bool colored = false;
    if (lane == 0) {
        if (a.C[v] != GC_UNC) flag_error(a, 3, k, v);
        colored = settle(v, rs, r, f, k, a.C, a.W, a.P);
    }
    colored = __shfl_sync(kFull, colored, 0);
    colored_notify(a, colored && lane == 0, v, re - rs, k, !colored && lane == 0);
}

// One kSeg-entry segment of a long scan (whole warp); the warp finishing the
// last segment settles the vertex.
template <bool PROF>
__device__ __forceinline__ void scan_segment(const Args &a, uint32_t slot, uint32_t seg, uint32_t k,
                                             uint32_t &nvis) {
    const bool dense = k == 0;
    const unsigned lane = lane_id();
    const uint32_t thresh = 2u * k;
    // the slot was written by another SM in this phase: bypass L1 (a 128-byte
    // line holds four slots, so it may be cached from a neighbouring slot)
    LongScan *L = &a.LS[slot];
    const uint32_t v = __ldcg(&L->v);
    const uint32_t need = __ldcg(&L->need);
    const uint32_t Lbase = __ldcg(&L->base), Lsh = __ldcg(&L->sh), Lsl = __ldcg(&L->sl);
    if ((need >> 2) != k) {  // trap: slot written by another round
        if (lane == 0) flag_error(a, 15, k, (need >> 2));
        return;
    }
    if (v >= (uint32_t)a.n) {
        if (lane == 0) flag_error(a, 11, k, v);
        return;
    }
    const int64_t rs = a.ro[v], re = a.ro[v + 1];
    const int64_t e0 = rs + (int64_t)Lbase + (int64_t)seg * kSeg;
    const int64_t e1 = min(re, e0 + (int64_t)kSeg);
    if (e0 >= re) {
        if (lane == 0) flag_error(a, 12, k, v);
        return;
    }
    const uint32_t pv = weight_mix(v ^ a.key);
    // skip when every needed side already has a hit before this segment
    const uint32_t curH = *(volatile uint32_t *)&L->minH, curL = *(volatile uint32_t *)&L->minL;
    const uint32_t rel0 = (uint32_t)(e0 - rs);
    const bool want_hi = (need & 1u) && !(curH != kNone && curH < rel0);
    const bool want_lo = (need & 2u) && !(curL != kNone && curL < rel0);
    if (want_hi || want_lo) {
        uint32_t u[kSeg / 32], c[kSeg / 32];
#pragma unroll
        for (int q = 0; q < kSeg / 32; ++q) {
            const int64_t e = e0 + q * 32 + lane;
            u[q] = e < e1 ? a.ci[e] : 0u;
        }
#pragma unroll
        for (int q = 0; q < kSeg / 32; ++q) {
            const int64_t e = e0 + q * 32 + lane;
            c[q] = e < e1 ? __ldcg(&a.C[u[q]]) : 0u;
        }
        uint32_t rh = kNone, rl = kNone;
#pragma unroll
        for (int q = 0; q < kSeg / 32; ++q) {
            const int64_t e = e0 + q * 32 + lane;
            if (e < e1 && c[q] >= thresh) {
                const uint32_t pu = weight_mix(u[q] ^ a.key);
                const uint32_t rel = (uint32_t)(e - rs);
                if (want_hi && rel >= Lsh && pu > pv) rh = min(rh, rel);
                if (want_lo && rel >= Lsl && pu < pv) rl = min(rl, rel);
            }
        }
        if (PROF) {
            const int64_t cnt = e1 - e0 - (int64_t)lane;
            nvis += cnt > 0 ? (uint32_t)((cnt + 31) / 32) : 0u;
        }
        rh = __reduce_min_sync(kFull, rh);
        rl = __reduce_min_sync(kFull, rl);
        if (lane == 0) {
            if (rh != kNone) atomicMin(&L->minH, rh);
            if (rl != kNone) atomicMin(&L->minL, rl);
        }
    }
    bool last = false;
    if (lane == 0) {
        __threadfence();
        const uint32_t old = atomicSub(&L->ticket, 1u);
        if (old == 0u || old > 0x7FFFFFFFu) flag_error(a, 41, k, v);
        last = old == 1u;
    }
    last = __shfl_sync(kFull, last, 0);
    if (!last) return;
    bool colored = false;
    if (lane == 0) {
        __threadfence();
        const uint32_t mH = atomicAdd(&L->minH, 0u), mL = atomicAdd(&L->minL, 0u);
        const uint32_t deg = (uint32_t)(re - rs);
        const bool bad = (mH != kNone && mH >= deg) || (mL != kNone && mL >= deg);
        if (bad) {
            flag_error(a, (mH != kNone && mH >= deg) ? 13 : 14, k, v);
            a.ctr[47] = deg;
            a.ctr[48] = ((unsigned long long)mH << 32) | mL;
            a.ctr[49] = ((unsigned long long)Lbase << 32) | (need & 3u);
        }
        const Resume r = resume_of(v, rs, dense, a.W, a.P, a.C, thresh);
        Found f;
        if (mH != kNone && !bad) {
            f.hpos = rs + mH;
            f.hw = a.ci[f.hpos];
        }
        if (mL != kNone && !bad) {
            f.lpos = rs + mL;
            f.lw = a.ci[f.lpos];
        }
        if (a.C[v] != GC_UNC) flag_error(a, 4, k, v);
        if (!bad) colored = settle(v, rs, r, f, k, a.C, a.W, a.P);
        atomicExch(&a.owner[slot], k << 1);
    }
    colored = __shfl_sync(kFull, colored, 0);
    colored_notify(a, colored && lane == 0, v, re - rs, k, !colored && lane == 0);
}

// NOTIFY work of vertex u coloured in round k-1, processed in round k: wake
// the uncoloured neighbours that used u as a witness (round stamp k) and queue
// their evaluation.  This lane's entries: e0, e0 + stride, ... (< re).
template <int Q>
__device__ __forceinline__ void notify_entries(const Args &a, uint32_t u, int64_t e0, int64_t re,
                                               int stride, uint32_t k) {
    uint32_t w[Q], cw[Q];
    uint2 ww[Q];
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        const int64_t e = e0 + (int64_t)q * stride;
        w[q] = e < re ? a.ci[e] : kNone;
    }
#pragma unroll
    for (int q = 0; q < Q; ++q) cw[q] = w[q] != kNone ? __ldcg(&a.C[w[q]]) : 0u;
#pragma unroll
    for (int q = 0; q < Q; ++q) ww[q] = cw[q] == GC_UNC ? __ldcg(&a.W[w[q]]) : make_uint2(kNone, kNone);
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        bool wk = cw[q] == GC_UNC && (ww[q].x == u || ww[q].y == u);
        if (wk) wk = atomicMax(&a.S[w[q]], k) < k;
        const unsigned m = __ballot_sync(kFull, wk);
        if (!m) continue;
        const unsigned leader = __ffs(m) - 1;
        unsigned long long b = 0;
        if (lane_id() == leader) {
            b = atomicAdd(QC(a, k & 1, qTail), (unsigned long long)__popc(m));
            atomicAdd(QC(a, k & 1, qEval), (unsigned long long)__popc(m));
        }
        b = __shfl_sync(kFull, b, leader);
        if (wk)
            put_item(a, k & 1, b + __popc(m & ((1u << lane_id()) - 1u)), make_uint2(w[q], T_EVAL << 28),
                     k);
    }
}

template <bool PROF>
__device__ __forceinline__ void process_item(const Args &a, uint2 it, uint32_t k, uint32_t &nvisE,
                                             uint32_t &nvisS, uint32_t &nvisN) {
    const uint32_t type = it.y >> 28, sub = it.y & kSub;
    const unsigned lane = lane_id();
    if (type == T_EVAL) {
        if (lane == 0 && atomicAdd(&a.S[it.x], 0u) != k) flag_error(a, 40, k, it.x);
        eval_warp<PROF>(a, it.x, k, nvisE);
    } else if (type == T_SCAN) {
        if (it.x >= *QC(a, k & 1, qLS)) {
            if (lane == 0) flag_error(a, 42, k, it.x);
            return;
        }
        scan_segment<PROF>(a, it.x, sub, k, nvisS);
    } else if (type == T_NOTIFY) {
        const uint32_t u = it.x;
        int64_t rs = a.ro[u], re = a.ro[u + 1];
        if (sub != kSub) {  // segment of a long row
            rs += (int64_t)sub * kNotifySeg;
            re = min(re, rs + (int64_t)kNotifySeg);
            notify_entries<kNotifySeg / 32>(a, u, rs + lane, re, 32, k);
        } else {            // whole short row (<= kLaneNotify entries)
            notify_entries<1>(a, u, rs + lane, re, 32, k);
        }
        if (PROF && lane == 0) nvisN += (uint32_t)(re - rs);
    } else if (lane == 0) {
        flag_error(a, 20, k, it.y);
    }
}

template <bool PROF>
__global__ void __launch_bounds__(kThreads, 2) k_event_persistent(Args a) {
    const unsigned lane = lane_id();
    const unsigned long long gtid = (unsigned long long)blockIdx.x * blockDim.x + threadIdx.x;
    const unsigned long long nthreads = (unsigned long long)gridDim.x * blockDim.x;
    const unsigned long long gwarp = gtid >> 5, nwarps = nthreads >> 5;
    uint32_t nvisE = 0, nvisS = 0, nvisN = 0;
    unsigned long long t0 = gtimer(), tacc[4] = {0, 0, 0, 0};
    uint32_t k = 0;

    // ------------------------------------------- static rounds 0 and 1
    // round 0: every vertex (dense); round 1: the vertices round 0 left
    // blocked, each re-checking its two witnesses.  Phases: lane windows ->
    // warp windows -> long-scan segments.
    bool finished = false;
    for (k = 0; k < 2; ++k) {
        const unsigned long long rem = (unsigned long long)a.n - a.ctr[kColTotal];
        if (gtid == 0 && (int64_t)k < a.nk_cap) a.nk[k] = (int64_t)rem;
        if (rem == 0) {
            finished = true;
            break;
        }
        const bool dense = k == 0;
        const uint32_t thresh = 2u * k;
        const unsigned long long N = dense ? (unsigned long long)a.n : a.ctr[r0B];
        if (PROF && gtid == 0 && (int64_t)k < a.nk_cap) a.rstat[4 * k] = (int64_t)N;
        for (unsigned long long base = gwarp * 32; base < N; base += nthreads) {
            const unsigned long long idx = base + lane;
            const bool valid = idx < N;
            uint32_t v = 0;
            int64_t rs = 0, re = 0;
            Resume r{false, false, 0, 0};
            if (valid) {
                v = dense ? (uint32_t)idx : a.B0[idx];
                rs = a.ro[v];
                re = a.ro[v + 1];
                r = resume_of(v, rs, dense, a.W, a.P, a.C, thresh);
            }
            const bool work = valid && (r.need_hi || r.need_lo);
            int64_t s = r.need_hi ? r.sh : re;
            if (r.need_lo && r.sl < s) s = r.sl;
            const int64_t lim = min(re, s + (int64_t)kLaneWin);
            Found f;
            if (work) lane_window<kLaneWin>(a, thresh, weight_mix(v ^ a.key), r, s, lim, f);
            if (PROF && work) nvisE += (uint32_t)(lim - s);
            const bool unresolved =
                work && lim < re && ((r.need_hi && f.hpos < 0) || (r.need_lo && f.lpos < 0));
            bool colored = false;
            if (work && !unresolved) colored = settle(v, rs, r, f, k, a.C, a.W, a.P);
            warp_append(unresolved, v, a.WQ0, &a.ctr[r0WQ + 3 * k]);
            colored_notify(a, colored, v, re - rs, k, work && !unresolved && !colored);
        }
        if (!grid_barrier(a, 0, k, -1)) return;
        const unsigned long long nwq = a.ctr[r0WQ + 3 * k];
        for (unsigned long long i = gwarp; i < nwq; i += nwarps) eval_warp<PROF>(a, a.WQ0[i], k, nvisE);
        if (!grid_barrier(a, 1, k, -1)) return;
        const unsigned long long nsq = a.ctr[r0SQ + 3 * k];
        for (unsigned long long i = gwarp; i < nsq; i += nwarps) {
            const uint2 it = a.SQ0[i];
            scan_segment<PROF>(a, it.x, it.y, k, nvisS);
        }
        if (!grid_barrier(a, 2, k, -1)) return;
        if (a.ctr[kErrPar + (k & 1)] != 0) {
            finished = true;
            break;
        }
    }
    if (PROF && gtid == 0) {
        const unsigned long long t = gtimer();
        tacc[0] += t - t0;
        t0 = t;
    }

    // -------------------------------------------------------- rounds >= 2
    for (k = 2; !finished; ++k) {
        const unsigned long long rem = (unsigned long long)a.n - a.ctr[kColTotal];
        if (gtid == 0 && (int64_t)k < a.nk_cap) a.nk[k] = (int64_t)rem;
        if (rem == 0 || k >= a.max_rounds) break;
        if (a.ctr[kErrPar + ((k - 1) & 1)] != 0) break;  // a trap fired (grid-uniform)
        const int qset = (int)(k & 1);
        uint2 *Qk = a.Q[k & 1];
        if (PROF && gtid == 0 && (int64_t)k < a.nk_cap) a.rstat[4 * k + 3] = (int64_t)*QC(a, qset, qTail);
        unsigned long long base0 = 0;  // first index served by the dynamic loop
        if (a.split) {
            // debug / A-B: the NOTIFY(k-1) items (the static prefix) first,
            // statically, then a barrier, then the EVAL / SCAN items they made
            const unsigned long long ns = *QC(a, qset, qTail);
            for (unsigned long long i = gwarp; i < ns; i += nwarps) {
                volatile uint2 *src = reinterpret_cast<volatile uint2 *>(&Qk[i]);
                const uint2 it = make_uint2(src->x, src->y);
                process_item<PROF>(a, it, k, nvisE, nvisS, nvisN);
                __syncwarp();
                if (lane == 0) Qk[i] = make_uint2(0u, 0u);
            }
            if (!grid_barrier(a, 4, k, -1)) return;
            base0 = ns;
        }
        // dynamic queue: claim, wait for publication, process, mark done.
        // A round has ~10^4 items; kDynWarps warps are plenty, the others go
        // straight to the barrier instead of polling the queue counters.
        for (; gwarp < a.dyn_warps;) {
            unsigned long long idx = 0;
            if (lane == 0) idx = base0 + atomicAdd(QC(a, qset, qHead), 1ull);
            idx = __shfl_sync(kFull, idx, 0);
            unsigned ix = 0, iy = 0;
            int state = 0;  // 1: item, 2: phase over, 3: timeout / abort
            if (lane == 0) {
                const unsigned long long tw0 = gtimer();
                unsigned backoff = 32;
                for (;;) {
                    const unsigned long long d = ld_acquire(QC(a, qset, qDone));
                    const unsigned long long t = ld_acquire(QC(a, qset, qTail));
                    if (idx < t) {
                        volatile uint2 *src = reinterpret_cast<volatile uint2 *>(&Qk[idx]);
                        while ((iy = src->y) == 0u)
                            if (gtimer() - tw0 > kBarrierTimeoutNs) break;
                        __threadfence();
                        ix = src->x;
                        state = iy ? 1 : 3;
                        break;
                    }
                    if (d + base0 == t) {
                        state = 2;
                        break;
                    }
                    if (*(volatile unsigned long long *)&a.ctr[kAbort] ||
                        gtimer() - tw0 > kBarrierTimeoutNs) {
                        state = 3;
                        break;
                    }
                    __nanosleep(backoff);
                    backoff = min(backoff * 2u, 1024u);
                }
            }
            state = __shfl_sync(kFull, state, 0);
            if (state == 2) break;
            if (state == 3) {
                if (lane == 0) {
                    flag_error(a, 30, k, (uint32_t)idx);
                    atomicExch(a.ctr + kAbort, 1ull);
                }
                break;
            }
            const uint2 it = make_uint2(__shfl_sync(kFull, ix, 0), __shfl_sync(kFull, iy, 0));
            process_item<PROF>(a, it, k, nvisE, nvisS, nvisN);
            __syncwarp();
            if (lane == 0) {
                Qk[idx] = make_uint2(0u, 0u);  // clean slot for the round after next
                __threadfence();
                atomicAdd(QC(a, qset, qDone), 1ull);
            }
        }
        if (PROF && gtid == 0 && (int64_t)k < a.nk_cap) {
            a.rstat[4 * k] = (int64_t)*QC(a, qset, qEval);
            a.rstat[4 * k + 2] = (int64_t)*QC(a, qset, qLS);
        }
        // the next phase pushes its NOTIFY items into set (k+2)&1 == k&1: reset it
        if (!grid_barrier(a, 3, k, (int)(k & 1))) return;
        if (PROF && gtid == 0) {
            const unsigned long long t = gtimer();
            tacc[1] += t - t0;
            t0 = t;
        }
    }
    if (gtid == 0) {
        a.ctr[kRem] = (unsigned long long)a.n - a.ctr[kColTotal];
        a.ctr[kRounds] = k;
        if (PROF)
            for (int i = 0; i < 4; ++i) a.ctr[kPhaseNs + i] = tacc[i];
    }
    if (PROF) {
        const unsigned e = __reduce_add_sync(kFull, nvisE);
        const unsigned s = __reduce_add_sync(kFull, nvisS);
        const unsigned q = __reduce_add_sync(kFull, nvisN);
        if (lane == 0) {
            if (e) atomicAdd(&a.ctr[kVisE], (unsigned long long)e);
            if (s) atomicAdd(&a.ctr[kVisS], (unsigned long long)s);
            if (q) atomicAdd(&a.ctr[kVisN], (unsigned long long)q);
        }
    }
}

template <bool PROF>
int launch(gc_graph *g, Args &a, int *blocks_out) {
    int per_sm = 0;
    GC_CUDA_TRY(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k_event_persistent<PROF>,
                                                              kThreads, 0));
    if (per_sm < 1) {
        set_error("persistent event kernel cannot be resident");
        return GC_ERR_CUDA;
    }
    const int blocks = per_sm * g->sm_count;
    void *args[] = {&a};
    GC_CUDA_TRY(cudaLaunchCooperativeKernel((void *)k_event_persistent<PROF>, blocks, kThreads, args,
                                            0, g->stream));
    *blocks_out = blocks;
    return GC_OK;
}

}  // namespace

int run_persistent_maxmin(gc_graph *g, const RunParams &p, RunResult *r) {
    Scratch &s = g->s;
    const int64_t n = g->n;
    r->rounds = r->inner = r->launches = 0;
    if (n == 0) return GC_OK;
    int rc = fill_u32(s.C, GC_UNC, n, g->stream);  // Alg.5 L5
    if (rc) return rc;
    GC_CUDA_TRY(cudaMemsetAsync(s.S, 0, sizeof(uint32_t) * (size_t)n, g->stream));
    GC_CUDA_TRY(cudaMemsetAsync(s.ctr, 0, 64 * sizeof(unsigned long long), g->stream));
    if (!s.qctl) GC_CUDA_TRY(cudaMalloc(&s.qctl, 256 * sizeof(unsigned long long)));
    GC_CUDA_TRY(cudaMemsetAsync(s.qctl, 0, 256 * sizeof(unsigned long long), g->stream));
    // per-round queue: NOTIFY items (<= n + m/128) + EVAL (<= n) + SCAN (<= n + m/256)
    const size_t qcap = (size_t)(3 * n + g->nnz / 64 + 64);
    if (s.Qd[0] == nullptr || s.qd_cap < qcap) {
        cudaFree(s.Qd[0]);
        cudaFree(s.Qd[1]);
        s.Qd[0] = s.Qd[1] = nullptr;
        GC_CUDA_TRY(cudaMalloc(&s.Qd[0], qcap * sizeof(uint2)));
        GC_CUDA_TRY(cudaMalloc(&s.Qd[1], qcap * sizeof(uint2)));
        s.qd_cap = qcap;
        GC_CUDA_TRY(cudaMemsetAsync(s.Qd[0], 0, qcap * sizeof(uint2), g->stream));
        GC_CUDA_TRY(cudaMemsetAsync(s.Qd[1], 0, qcap * sizeof(uint2), g->stream));
    }
    // (consumers zero every slot they read, so the queues stay clean across calls)
    // a round with >= 2 uncoloured vertices colours at least the global max
    // and min among them, so R <= n/2 + 1
    const int64_t max_rounds = std::min<int64_t>(std::min<int64_t>(p.max_rounds, 0xFFFFFFF0ll),
                                                 n / 2 + 2);
    rc = ensure_nk(g, std::min<int64_t>(std::min<int64_t>(n + 2, max_rounds + 2), 1 << 20));
    if (rc) return rc;
    Args a;
    a.ro = g->ro;
    a.ci = g->ci;
    a.C = s.C;
    a.W = reinterpret_cast<uint2 *>(s.W);
    a.P = reinterpret_cast<uint2 *>(s.P);
    a.S = s.S;
    a.WQ0 = s.hub;
    a.B0 = s.F[0];
    a.SQ0 = reinterpret_cast<uint2 *>(s.Q2);
    a.LS = reinterpret_cast<LongScan *>(s.LS);
    a.Q[0] = reinterpret_cast<uint2 *>(s.Qd[0]);
    a.qc = s.qctl;
    a.Q[1] = reinterpret_cast<uint2 *>(s.Qd[1]);
    a.ctr = s.ctr;
    a.nk = s.nk;
    a.rstat = s.rstat;
    a.nk_cap = s.nk_cap;
    a.n = n;
    a.key = p.keys.k[0];
    a.max_rounds = (uint32_t)max_rounds;
    a.q_cap = (unsigned long long)qcap;
    a.sq_cap = (unsigned long long)(n + g->nnz / 128 + 1);
    a.ls_cap = (unsigned long long)n;
    a.dyn_warps = p.dyn_warps > 0 ? (unsigned long long)p.dyn_warps : kDynWarps;
    a.split = p.split;
    a.owner = s.Q3;
    GC_CUDA_TRY(cudaMemsetAsync(s.Q3, 0, sizeof(uint32_t) * (size_t)n, g->stream));
    const bool prof = p.prof && p.prof->on;
    cudaEvent_t e0 = nullptr, e1 = nullptr;
    if (prof) {
        GC_CUDA_TRY(cudaEventCreate(&e0));
        GC_CUDA_TRY(cudaEventCreate(&e1));
        GC_CUDA_TRY(cudaEventRecord(e0, g->stream));
    }
    int blocks = 0;
    rc = prof ? launch<true>(g, a, &blocks) : launch<false>(g, a, &blocks);
    if (rc) return rc;
    r->launches += 2;  // fill + persistent kernel
    if (prof) GC_CUDA_TRY(cudaEventRecord(e1, g->stream));
    unsigned long long h[24];
    GC_CUDA_TRY(cudaMemcpyAsync(h, s.ctr + kRem, sizeof(h), cudaMemcpyDeviceToHost, g->stream));
    GC_CUDA_TRY(cudaStreamSynchronize(g->stream));
    if (h[kErr - kRem] != 0) {
        char buf[160];
        snprintf(buf, sizeof(buf),
                 "internal consistency check %llu failed in round %llu (%llu) dbg %llu %llx %llx",
                 h[kErr - kRem], h[kErr - kRem + 1], h[kErr - kRem + 2], h[7], h[8], h[9]);
        set_error(buf);
        return GC_ERR_CUDA;
    }
    if (h[0] != 0) {
        set_error("max-min colouring exceeded the round limit");
        return GC_ERR_TOO_LARGE;
    }
    r->rounds = (int64_t)h[kRounds - kRem];
    r->inner = r->rounds;
    if (prof) {
        float ms = 0.f;
        cudaEventElapsedTime(&ms, e0, e1);
        cudaEventDestroy(e0);
        cudaEventDestroy(e1);
        p.prof->ms[0] += ms;
        p.prof->launches[0] += 1;
        p.prof->launch_us.push_back(1e3f * ms);
        // phase split (globaltimer, thread 0): [1] rounds 0-1, [2] rounds >= 2
        p.prof->ms[1] += (double)h[kPhaseNs - kRem] / 1e6;
        p.prof->ms[2] += (double)h[kPhaseNs + 1 - kRem] / 1e6;
        const int64_t visE = (int64_t)h[kVisE - kRem], visS = (int64_t)h[kVisS - kRem],
                      visN = (int64_t)h[kVisN - kRem];
        // evaluations: every vertex in round 0, the blocked ones in round 1,
        // then the woken ones
        int64_t sumD = n;
        if (r->rounds > 1) {
            const int64_t m = std::min<int64_t>(r->rounds, s.nk_cap);
            std::vector<int64_t> rs((size_t)4 * m, 0);
            GC_CUDA_TRY(cudaMemcpy(rs.data(), s.rstat, sizeof(int64_t) * 4 * m, cudaMemcpyDeviceToHost));
            for (int64_t kk = 1; kk < m; ++kk) sumD += rs[4 * kk];
        }
        // algorithmic bytes: per evaluated vertex 16 B row
        // offsets + (rounds >= 1) 8 B queue item + 16 B witness state + 16 B
        // state write; 8 B colour + item per coloured vertex; 4 B per scanned
        // entry; per coloured vertex 20 B + 4 B per notified entry.
        const int64_t b = 16 * sumD + 8 * (sumD - n) + 16 * (sumD - n) + 16 * (sumD - n) + 8 * n +
                          4 * (visE + visS) + 20 * n + 4 * visN;
        p.prof->bytes[0] += b;
        p.prof->visits += visE + visS;
    }
    return GC_OK;
}

}  // namespace gc
