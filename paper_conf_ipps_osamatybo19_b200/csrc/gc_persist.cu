// gc_persist.cu -- EVENT mode as ONE persistent cooperative kernel that runs
// every round of the max-min colouring (Alg.1 + Alg.5, P:L102-113,
// P:L506-556; H = 1) with grid-wide barriers instead of kernel boundaries.
//
// The method per round is the witness/resume scheme of gc_event.cu; this file
// only changes how the work of a round is scheduled on the 148 SMs:
//   P1  evaluate D_k: one lane per vertex (round 0 and large D_k: scan a
//       window of kLaneWin entries, unresolved rows go to WQ) or one warp per
//       vertex (scan a kWarpWin window, unresolved rows become long scans);
//   P1b WQ: one warp per vertex, same as the warp path of P1;
//   P2  long scans split into kSeg-entry segments over all warps; each segment
//       atomicMin's its first hi / lo hit into the scan's slot, and the warp
//       finishing the last segment settles the vertex (first-hit semantics are
//       kept, so the cursor invariant holds);
//   P3  notify: rows of vertices coloured in this round -- short rows one lane
//       each, long rows as kNotifySeg-entry segments over all warps -- wake the
//       uncoloured neighbours that used the coloured vertex as a witness.
// A phase whose queue is empty is skipped (its barrier too): the decision is
// taken after a barrier from device counters, so it is grid-uniform.
// The host launches one kernel per colouring; per-round sizes land in nk[].

#include <cstdio>
#include <cstdlib>

#include "gc_event_common.cuh"


namespace gc {

int fill_u32(uint32_t *p, uint32_t val, int64_t n, cudaStream_t st);
int ensure_nk(gc_graph *g, int64_t need);

namespace {

using namespace ev;

constexpr int kThreads = 1024;  // one block per SM: fewer barrier arrivals
constexpr int kLaneWin = 8;      // entries a lane scans before handing off
constexpr int kWarpWin = 256;    // entries a warp scans before splitting
constexpr int kSeg = 256;        // entries per long-scan segment (8 per lane)
constexpr int kNotifySeg = 128;  // entries per notify segment (4 per lane)
constexpr int kLaneNotify = 32;  // rows up to this length are notified by one lane

// counter layout: two sets of 8 (by round parity) at ctr[24..39]
enum : int { cD = 0, cWQ = 1, cSQ = 2, cLS = 3, cNQS = 4, cNQ = 5, cI = 6 };
enum : int {
    kSet = 24,
    kRem = 40,
    kVisE = 41,
    kVisS = 42,
    kVisN = 43,
    kSumD = 44,
    kRounds = 45,
    kPhaseNs = 50  // [50..53] PROF: ns spent in P1, P1b+P2, P3, barriers
};

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
    uint32_t *M;     // bit u set iff u was uncoloured at the start of this round
    uint32_t *D[2];
    uint32_t *WQ;
    uint2 *SQ;
    LongScan *LS;
    uint32_t *NQS;
    uint2 *NQ;
    unsigned long long *ctr;
    int64_t *nk;
    int64_t *rstat;
    int64_t nk_cap;
    int64_t n;
    uint32_t key;
    uint32_t max_rounds;
    unsigned long long nq_cap, sq_cap, ls_cap;  // queue capacities (items)
    unsigned long long *hist;  // PROF + GC_PROFILE_HIST: [8][32] log2 histograms, else null
};

// Internal-consistency trap: record the first violation (kind, round, vertex)
// in ctr[kErr..kErr+2] instead of writing out of bounds.
// ctr[kErrPar + (k & 1)] marks "a trap fired in round k"; it is read at the
// top of round k+1, after the barrier, so the exit decision is grid-uniform.
enum : int { kErr = 56, kErrPar = 59 };
__device__ __forceinline__ void flag_error(const Args &a, unsigned kind, uint32_t k, uint32_t v) {
    if (atomicCAS(&a.ctr[kErr], 0ull, (unsigned long long)kind) == 0ull) {
        a.ctr[kErr + 1] = k;
        a.ctr[kErr + 2] = v;
    }
    a.ctr[kErrPar + (k & 1)] = 1;
}

// Round-start status (the snapshot of Alg.5 L26, R6) as a 2 MB-per-16M-vertex
// bitmask that stays in L2: bits are cleared in P3 for the vertices coloured
// in the round, so the scans of P1 / P2 read exactly the round-start state and
// colours written concurrently in the round still count as uncoloured.
__device__ __forceinline__ bool active(const Args &a, uint32_t u) {
    return (a.M[u >> 5] >> (u & 31)) & 1u;
}

// Where a vertex resumes (cf. gc_event_common resume_of, with the bitmask).
__device__ __forceinline__ Resume resume_m(const Args &a, uint32_t v, int64_t rs, bool dense) {
    Resume r;
    if (dense) {
        r.need_hi = r.need_lo = true;
        r.sh = r.sl = rs;
    } else {
        const uint2 w = a.W[v];
        const uint2 p = a.P[v];
        r.need_hi = !active(a, w.x);  // hi witness coloured in an earlier round
        r.need_lo = !active(a, w.y);
        r.sh = rs + (int64_t)p.x + 1;
        r.sl = rs + (int64_t)p.y + 1;
    }
    return r;
}

__device__ __forceinline__ unsigned long long gtimer() {
    unsigned long long t;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
    return t;
}

// Grid-wide phase boundary (the kernel is launched cooperatively, so every
// block is resident).  Monotone arrival counter on ctr[kBar].  A wait longer
// than kBarrierTimeoutNs records a trap and makes every block leave the
// kernel (returns false) instead of hanging the GPU.  The waiting thread then
// issues a gpu-scope fence, which also invalidates its SM's L1 (CCTL.IVALL):
// the next phase reads state other SMs wrote, and L1 is not coherent.
enum : int { kBar = 61, kAbort = 63 };
constexpr unsigned long long kBarrierTimeoutNs = 4000000000ull;

__device__ __forceinline__ unsigned long long ld_acquire(const unsigned long long *p) {
    unsigned long long v;
    asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}

// release-ordered arrival (MEMBAR.ALL.GPU + atomic; a __threadfence is the
// much slower sequentially consistent MEMBAR.SC.GPU) and acquire-ordered
// loads (which also invalidate this SM's L1: CCTL.IVALL)
__device__ __forceinline__ unsigned long long atom_add_release(unsigned long long *p,
                                                               unsigned long long x) {
    unsigned long long v;
    asm volatile("atom.add.release.gpu.global.u64 %0, [%1], %2;" : "=l"(v) : "l"(p), "l"(x) : "memory");
    return v;
}
__device__ __forceinline__ uint32_t atom_sub_acq_rel(uint32_t *p, uint32_t x) {
    uint32_t v;
    asm volatile("atom.add.acq_rel.gpu.global.u32 %0, [%1], %2;" : "=r"(v) : "l"(p), "r"(0u - x) : "memory");
    return v;
}

__device__ __forceinline__ bool phase_barrier(const Args &a, int id, uint32_t k) {
    __shared__ int ok_sh;
    __syncthreads();
    if (threadIdx.x == 0) {
        // monotone arrival counter: barrier instance i completes when it
        // reaches (i + 1) * gridDim.x -- one atomic per block, no reset
        int ok = 1;
        const unsigned long long old = atom_add_release(a.ctr + kBar, 1ull);
        const unsigned long long target = (old / gridDim.x + 1) * gridDim.x;
        unsigned spins = 0;
        const unsigned long long t0 = gtimer();
        while (ld_acquire(a.ctr + kBar) < target) {
            if ((++spins & 255u) == 0u) {
                if (*(volatile unsigned long long *)(a.ctr + kAbort)) {
                    ok = 0;
                    break;
                }
                if (gtimer() - t0 > kBarrierTimeoutNs) {
                    flag_error(a, 100 + id, k, blockIdx.x);
                    atomicExch(a.ctr + kAbort, 1ull);
                    ok = 0;
                    break;
                }
            }
        }
        ok_sh = ok;  // the acquire loads of the spin invalidated this SM's L1
    }
    __syncthreads();
    return ok_sh != 0;
}

// ---------------------------------------------------------------- staging
// Appends to the shared lists (coloured rows to notify, woken vertices,
// overflowing lane windows) and the coloured count are staged per block in
// shared memory and flushed with ONE global atomic per list per block at the
// end of each phase: with a warp per vertex every colouring would otherwise
// be 2-3 global atomics on one cache line, serialised in one L2 slice.  A
// list that overflows its shared buffer falls back to global appends.
constexpr int kStNQS = 4096, kStNQ = 4096, kStD = 8192, kStWQ = 4096;
struct Stage {
    uint32_t nqs[kStNQS];
    uint2 nq[kStNQ];
    uint32_t d[kStD];
    uint32_t wq[kStWQ];
    unsigned n[4];            // staged counts: 0 nqs, 1 nq, 2 d, 3 wq
    unsigned colored;         // staged coloured count
    unsigned long long base[4];
};
constexpr size_t kStageBytes = sizeof(Stage);

__device__ __forceinline__ Stage &stage() {
    extern __shared__ __align__(16) unsigned char smem_raw[];
    return *reinterpret_cast<Stage *>(smem_raw);
}

// Whole warp converged: lanes with `pred` append make(lane) to staged list
// `li` (shared buffer buf of capacity cap), spilling to the global list /
// counter beyond the capacity.
template <class T>
__device__ __forceinline__ void stage_append(bool pred, T val, int li, T *buf, int cap, T *glist,
                                             unsigned long long *gcount) {
    const unsigned m = __ballot_sync(kFull, pred);
    if (!m) return;
    Stage &st = stage();
    const unsigned lane = lane_id();
    const unsigned leader = __ffs(m) - 1;
    unsigned base = 0;
    if (lane == leader) base = atomicAdd(&st.n[li], (unsigned)__popc(m));
    base = __shfl_sync(kFull, base, leader);
    const unsigned pos = base + __popc(m & ((1u << lane) - 1u));
    const bool spill = pred && pos >= (unsigned)cap;
    if (pred && !spill) buf[pos] = val;
    const unsigned sm = __ballot_sync(kFull, spill);
    if (sm) {
        const unsigned sl = __ffs(sm) - 1;
        unsigned long long gb = 0;
        if (lane == sl) gb = atomicAdd(gcount, (unsigned long long)__popc(sm));
        gb = __shfl_sync(kFull, gb, sl);
        if (spill) glist[gb + __popc(sm & ((1u << lane) - 1u))] = val;
    }
}

// Whole block, at the end of a phase: move the staged entries to the global
// lists (one atomicAdd per non-empty list) and add the coloured count.
// PROF: log2 histogram row `row` of a.hist (rows 0-3: cycles of one segment
// scan / settle of a long scan / warp evaluation / notify segment; rows 4-7:
// ns of one block's work in phase P1 / P1b / P2 / P3)
__device__ __forceinline__ void prof_hist(const Args &a, int row, unsigned long long x) {
    if (!a.hist) return;
    const int b = x ? min(31, 63 - __clzll((long long)x)) : 0;
    atomicAdd(&a.hist[row * 32 + b], 1ull);
}

__device__ __forceinline__ void stage_flush(const Args &a, unsigned long long *cs,
                                            unsigned long long *dcount, uint32_t *Dout,
                                            unsigned long long *prof_slot = nullptr,
                                            unsigned long long phase_t0 = 0, int phase = 0) {
    Stage &st = stage();
    __syncthreads();
    if (prof_slot && threadIdx.x == 0) {
        const unsigned long long dt = gtimer() - phase_t0;
        atomicMax(prof_slot, dt);
        prof_hist(a, 4 + phase, dt);
    }
    if (threadIdx.x == 0) {
        unsigned long long *ctrs[4] = {&cs[cNQS], &cs[cNQ], dcount, &cs[cWQ]};
        const int caps[4] = {kStNQS, kStNQ, kStD, kStWQ};
        for (int i = 0; i < 4; ++i) {
            const unsigned c = min(st.n[i], (unsigned)caps[i]);
            st.n[i] = c;
            st.base[i] = c ? atomicAdd(ctrs[i], (unsigned long long)c) : 0ull;
        }
        if (st.colored) atomicAdd(&cs[cI], (unsigned long long)st.colored);
        st.colored = 0;
    }
    __syncthreads();
    for (unsigned i = threadIdx.x; i < st.n[0]; i += blockDim.x) a.NQS[st.base[0] + i] = st.nqs[i];
    for (unsigned i = threadIdx.x; i < st.n[1]; i += blockDim.x) a.NQ[st.base[1] + i] = st.nq[i];
    for (unsigned i = threadIdx.x; i < st.n[2]; i += blockDim.x) Dout[st.base[2] + i] = st.d[i];
    for (unsigned i = threadIdx.x; i < st.n[3]; i += blockDim.x) a.WQ[st.base[3] + i] = st.wq[i];
    __syncthreads();
    if (threadIdx.x < 4) st.n[threadIdx.x] = 0;
    // (the barrier that follows starts with __syncthreads)
}

// Enqueue the notification work of lanes whose vertex was just coloured
// (whole warp converged).  Short rows -> NQS (one lane each); long rows ->
// NQ segments.
__device__ __forceinline__ void enqueue_notify(const Args &a, unsigned long long *cs, bool colored,
                                               uint32_t u, int64_t deg, uint32_t k) {
    Stage &st = stage();
    const bool shortrow = colored && deg <= kLaneNotify;
    stage_append<uint32_t>(shortrow, u, 0, st.nqs, kStNQS, a.NQS, &cs[cNQS]);
    unsigned lm = __ballot_sync(kFull, colored && !shortrow);
    while (lm) {  // long rows: the whole warp stages the segment items
        const int src = __ffs(lm) - 1;
        lm &= lm - 1;
        const uint32_t uu = __shfl_sync(kFull, u, src);
        const int64_t dg = __shfl_sync(kFull, deg, src);
        const uint32_t nseg = (uint32_t)((dg + kNotifySeg - 1) / kNotifySeg);
        for (uint32_t q0 = 0; q0 < nseg; q0 += 32) {
            const uint32_t q = q0 + lane_id();
            stage_append<uint2>(q < nseg, make_uint2(uu, q), 1, st.nq, kStNQ, a.NQ, &cs[cNQ]);
        }
    }
    const unsigned m = __ballot_sync(kFull, colored);
    if (m && lane_id() == (unsigned)(__ffs(m) - 1)) atomicAdd(&st.colored, (unsigned)__popc(m));
}

// Whole-warp first-hit search of a window [s, lim) of at most kWarpWin
// entries, issued in one shot: every lane loads its 8 column indices, then
// the 8 colours, then the hits are resolved in entry order (entry e0 + 32 q +
// lane) with one ballot per 32-entry row -- two dependent load steps instead
// of one pair per 64 entries.
__device__ __forceinline__ void warp_window(const Args &a, uint32_t thresh, uint32_t pv,
                                            const Resume &r, int64_t s, int64_t lim, Found &f,
                                            uint32_t &nvis) {
    constexpr int Q = kWarpWin / 32;
    const unsigned lane = lane_id();
    uint32_t u[Q], c[Q];
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        const int64_t e = s + q * 32 + lane;
        u[q] = e < lim ? a.ci[e] : 0u;
    }
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        const int64_t e = s + q * 32 + lane;
        c[q] = e < lim ? (uint32_t)active(a, u[q]) : 0u;
    }
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        const int64_t e = s + q * 32 + lane;
        nvis += e < lim;
        bool h = false, l = false;
        if (e < lim && c[q]) {
            const uint32_t pu = weight_mix(u[q] ^ a.key);
            h = r.need_hi && e >= r.sh && pu > pv;
            l = r.need_lo && e >= r.sl && pu < pv;
        }
        const unsigned bh = __ballot_sync(kFull, h), bl = __ballot_sync(kFull, l);
        if (f.hpos < 0 && bh) {
            const int ln = __ffs(bh) - 1;
            f.hpos = s + q * 32 + ln;
            f.hw = __shfl_sync(kFull, u[q], ln);
        }
        if (f.lpos < 0 && bl) {
            const int ln = __ffs(bl) - 1;
            f.lpos = s + q * 32 + ln;
            f.lw = __shfl_sync(kFull, u[q], ln);
        }
    }
}

// PROF: longest single operation of a round (SM cycles), rstat[16k + 12 + i]
__device__ __forceinline__ void prof_max(const Args &a, uint32_t k, int i, long long cycles) {
    if ((int64_t)k < a.nk_cap && lane_id() == 0)
        atomicMax(reinterpret_cast<unsigned long long *>(a.rstat + 16 * k + 12 + i),
                  (unsigned long long)cycles);
    if (lane_id() == 0) prof_hist(a, i, (unsigned long long)cycles);
}

// Whole-warp evaluation of one vertex of D_k (warp-uniform arguments): scan a
// window; resolved -> settle; otherwise open a long scan (P2).
template <bool PROF>
__device__ __forceinline__ void eval_warp(const Args &a, unsigned long long *cs, uint32_t v,
                                          uint32_t k, bool dense, uint32_t &nvis) {
    const uint32_t thresh = 2u * k;
    const unsigned lane = lane_id();
    const int64_t rs = a.ro[v], re = a.ro[v + 1];
    const Resume r = resume_m(a, v, rs, dense);
    if (!r.need_hi && !r.need_lo) return;
    int64_t s = r.need_hi ? r.sh : re;
    if (r.need_lo && r.sl < s) s = r.sl;
    const int64_t lim = min(re, s + (int64_t)kWarpWin);
    Found f;
    uint32_t vis = 0;
    warp_window(a, thresh, weight_mix(v ^ a.key), r, s, lim, f, vis);
    if (PROF) nvis += vis;
    const bool miss_hi = r.need_hi && f.hpos < 0;
    const bool miss_lo = r.need_lo && f.lpos < 0;
    if (lim < re && (miss_hi || miss_lo)) {
        // long scan of [lim, re) for the missing sides
        const uint32_t nseg = (uint32_t)((re - lim + kSeg - 1) / kSeg);
        unsigned long long slot = 0, b = 0;
        if (lane == 0) {
            slot = atomicAdd(&cs[cLS], 1ull);
            b = atomicAdd(&cs[cSQ], (unsigned long long)nseg);
            if (slot >= a.ls_cap || b + nseg > a.sq_cap) {
                flag_error(a, 2, k, v);
                slot = ~0ull;
            }
        }
        slot = __shfl_sync(kFull, slot, 0);
        if (slot == ~0ull) return;
        if (lane == 0) {
            LongScan L;
            L.v = v;
            L.ticket = nseg;
            L.minH = f.hpos >= 0 ? (uint32_t)(f.hpos - rs) : kNone;
            L.minL = f.lpos >= 0 ? (uint32_t)(f.lpos - rs) : kNone;
            L.need = (miss_hi ? 1u : 0u) | (miss_lo ? 2u : 0u);
            L.sh = (uint32_t)(r.sh - rs);
            L.sl = (uint32_t)(r.sl - rs);
            L.base = (uint32_t)(lim - rs);
            a.LS[slot] = L;
        }
        b = __shfl_sync(kFull, b, 0);
        for (uint32_t q = lane; q < nseg; q += 32) a.SQ[b + q] = make_uint2((uint32_t)slot, q);
        return;
    }
    bool colored = false;
    if (lane == 0) {
        if (a.C[v] != GC_UNC) flag_error(a, 3, k, v);
        colored = settle(v, rs, r, f, k, a.C, a.W, a.P);
    }
    colored = __shfl_sync(kFull, colored, 0);
    enqueue_notify(a, cs, colored && lane == 0, v, re - rs, k);
}

// One kSeg-entry segment of a long scan (whole warp).
template <bool PROF>
__device__ __forceinline__ void scan_segment(const Args &a, unsigned long long *cs, uint2 item,
                                             uint32_t k, bool dense, uint32_t &nvis) {
    const unsigned lane = lane_id();
    const uint32_t thresh = 2u * k;
    if (item.x >= __ldcg(&cs[cLS])) {  // trap: segment of a slot not opened this round
        if (lane == 0) flag_error(a, 10, k, item.x);
        return;
    }
    LongScan *L = &a.LS[item.x];
    const uint32_t v = L->v;
    const uint32_t need = L->need;
    if (v >= (uint32_t)a.n) {
        if (lane == 0) flag_error(a, 11, k, v);
        return;
    }
    const int64_t rs = a.ro[v], re = a.ro[v + 1];
    const int64_t e0 = rs + (int64_t)L->base + (int64_t)item.y * kSeg;
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
            c[q] = e < e1 ? (uint32_t)active(a, u[q]) : 0u;
        }
        uint32_t rh = kNone, rl = kNone;
#pragma unroll
        for (int q = 0; q < kSeg / 32; ++q) {
            const int64_t e = e0 + q * 32 + lane;
            if (e < e1 && c[q]) {
                const uint32_t pu = weight_mix(u[q] ^ a.key);
                const uint32_t rel = (uint32_t)(e - rs);
                if (want_hi && rel >= L->sh && pu > pv) rh = min(rh, rel);
                if (want_lo && rel >= L->sl && pu < pv) rl = min(rl, rel);
            }
        }
        if (PROF) {
            const int64_t cnt = e1 - e0 - (int64_t)lane;  // this lane's entries in the segment
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
    if (lane == 0) last = atom_sub_acq_rel(&L->ticket, 1u) == 1u;
    last = __shfl_sync(kFull, last, 0);
    if (!last) return;
    const long long cf0 = PROF ? clock64() : 0;
    // the warp that finished the last segment settles v
    bool colored = false;
    if (lane == 0) {
        const uint32_t mH = atomicAdd(&L->minH, 0u), mL = atomicAdd(&L->minL, 0u);
        const bool bad = (mH != kNone && mH >= (uint32_t)(re - rs)) ||
                         (mL != kNone && mL >= (uint32_t)(re - rs));
        if (bad) flag_error(a, 13 + (mH != kNone && mH >= (uint32_t)(re - rs) ? 0 : 1), k, v);
        const Resume r = resume_m(a, v, rs, dense);
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
    }
    colored = __shfl_sync(kFull, colored, 0);
    enqueue_notify(a, cs, colored && lane == 0, v, re - rs, k);
    if (PROF) prof_max(a, k, 1, clock64() - cf0);
}

// Lane-serial search of a short window [s, lim) (lim - s <= WIN): all column
// indices first, then all colours, then the in-order first-hit test, so the
// lane waits for two dependent loads instead of 2 * WIN.
template <int WIN>
__device__ __forceinline__ void lane_window(const Args &a, uint32_t thresh, uint32_t pv,
                                            const Resume &r, int64_t s, int64_t lim, Found &f) {
    uint32_t u[WIN], c[WIN];
#pragma unroll
    for (int q = 0; q < WIN; ++q) u[q] = s + q < lim ? a.ci[s + q] : 0u;
#pragma unroll
    for (int q = 0; q < WIN; ++q) c[q] = s + q < lim ? (uint32_t)active(a, u[q]) : 0u;
#pragma unroll
    for (int q = 0; q < WIN; ++q) {
        const int64_t e = s + q;
        if (e < lim && c[q]) {
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

// Wake the neighbours at e0, e0+stride, ... (< re) of vertex u coloured in
// round k (whole warp converged; u == kNone for idle lanes).  Loads are issued
// level by level -- all column indices, then all colours, then the witnesses
// of the uncoloured ones -- so one lane's Q gathers overlap.
template <int Q>
__device__ __forceinline__ void notify_entries(const Args &a, uint32_t u, int64_t e0, int64_t re,
                                               int stride, uint32_t k, uint32_t *Dout,
                                               unsigned long long *dcount) {
    uint32_t w[Q], cw[Q];
    uint2 ww[Q];
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        const int64_t e = e0 + (int64_t)q * stride;
        w[q] = (u != kNone && e < re) ? a.ci[e] : kNone;
    }
    // colour and witnesses are loaded together (one dependent step, not two)
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        cw[q] = w[q] != kNone ? a.C[w[q]] : 0u;
        ww[q] = w[q] != kNone ? a.W[w[q]] : make_uint2(kNone, kNone);
    }
#pragma unroll
    for (int q = 0; q < Q; ++q) {
        bool wk = cw[q] == GC_UNC && (ww[q].x == u || ww[q].y == u);
        if (wk) wk = atomicMax(&a.S[w[q]], k + 1u) < k + 1u;
        stage_append<uint32_t>(wk, w[q], 2, stage().d, kStD, Dout, dcount);
    }
}

template <bool PROF>
__global__ void __launch_bounds__(kThreads, 1) k_event_persistent(Args a) {
    const unsigned lane = lane_id();
    const unsigned long long gtid = (unsigned long long)blockIdx.x * blockDim.x + threadIdx.x;
    const unsigned long long nthreads = (unsigned long long)gridDim.x * blockDim.x;
    const unsigned long long gwarp = gtid >> 5, nwarps = nthreads >> 5;
    unsigned long long rem = a.ctr[kRem];
    uint32_t nvisE = 0, nvisS = 0, nvisN = 0;
    unsigned long long t0 = 0, tacc[4] = {0, 0, 0, 0};
    uint32_t k = 0;
    {
        Stage &st = stage();
        if (threadIdx.x < 4) st.n[threadIdx.x] = 0;
        if (threadIdx.x == 0) st.colored = 0;
        __syncthreads();
    }
    for (;; ++k) {
        unsigned long long *cs = a.ctr + kSet + 8 * (k & 1);
        unsigned long long *cn = a.ctr + kSet + 8 * ((k + 1) & 1);
        if (gtid == 0 && (int64_t)k < a.nk_cap) a.nk[k] = (int64_t)rem;
        if (rem == 0 || k >= a.max_rounds) break;  // uniform: rem is computed identically
        if (k > 0 && __ldcg(&a.ctr[kErrPar + ((k - 1) & 1)]) != 0) break;  // a trap fired
        const bool dense = k == 0;
        const unsigned long long N = dense ? (unsigned long long)a.n : cs[cD];
        if (gtid == 0) {
            for (int i = 0; i < 8; ++i) cn[i] = 0;
            if (PROF) {
                a.ctr[kSumD] += N;
                if ((int64_t)k < a.nk_cap) a.rstat[16 * k] = (int64_t)N;
                t0 = gtimer();
            }
        }
        const uint32_t *Din = a.D[k & 1];
        uint32_t *Dout = a.D[(k + 1) & 1];
        unsigned long long *dcount = &cn[cD];
        // PROF: longest per-block work time of each phase -> rstat[16k + 8 + phase]
        unsigned long long tb = PROF ? gtimer() : 0ull;
        unsigned long long *pslot =
            (PROF && (int64_t)k < a.nk_cap) ? reinterpret_cast<unsigned long long *>(a.rstat + 16 * k + 8)
                                            : nullptr;
        const uint32_t thresh = 2u * k;
        // ------------------------------------------------------------ P1
        if (dense || N > 4 * nwarps) {
            for (unsigned long long base = gwarp * 32; base < N; base += nthreads) {
                const unsigned long long idx = base + lane;
                const bool valid = idx < N;
                uint32_t v = 0;
                int64_t rs = 0, re = 0;
                Resume r{false, false, 0, 0};
                if (valid) {
                    v = dense ? (uint32_t)idx : Din[idx];
                    rs = a.ro[v];
                    re = a.ro[v + 1];
                    r = resume_m(a, v, rs, dense);
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
                if (work && !unresolved) {
                    if (a.C[v] != GC_UNC) flag_error(a, 5, k, v);
                    colored = settle(v, rs, r, f, k, a.C, a.W, a.P);
                }
                stage_append<uint32_t>(unresolved, v, 3, stage().wq, kStWQ, a.WQ, &cs[cWQ]);
                enqueue_notify(a, cs, colored, v, re - rs, k);
            }
        } else {
            for (unsigned long long i = gwarp; i < N; i += nwarps) {
                const long long c0 = PROF ? clock64() : 0;
                eval_warp<PROF>(a, cs, Din[i], k, false, nvisE);
                if (PROF) prof_max(a, k, 2, clock64() - c0);
            }
        }
        stage_flush(a, cs, dcount, Dout, pslot ? pslot + 0 : nullptr, tb, 0);
        if (!phase_barrier(a, 0, k)) return;
        if (PROF) tb = gtimer();
        if (PROF && gtid == 0) {
            unsigned long long t = gtimer();
            tacc[0] += t - t0;
            if ((int64_t)k < a.nk_cap) a.rstat[16 * k + 4] = (int64_t)(t - t0);
            t0 = t;
        }
        // ----------------------------------------------------------- P1b
        const unsigned long long nwq = cs[cWQ];
        if (nwq) {
            for (unsigned long long i = gwarp; i < nwq; i += nwarps)
                eval_warp<PROF>(a, cs, a.WQ[i], k, dense, nvisE);
            stage_flush(a, cs, dcount, Dout, pslot ? pslot + 1 : nullptr, tb, 1);
            if (!phase_barrier(a, 1, k)) return;
            if (PROF) tb = gtimer();
        }
        // ------------------------------------------------------------ P2
        const unsigned long long nsq = cs[cSQ];
        if (nsq) {
            for (unsigned long long i = gwarp; i < nsq; i += nwarps) {
                const long long c0 = PROF ? clock64() : 0;
                scan_segment<PROF>(a, cs, a.SQ[i], k, dense, nvisS);
                if (PROF) prof_max(a, k, 0, clock64() - c0);
            }
            stage_flush(a, cs, dcount, Dout, pslot ? pslot + 2 : nullptr, tb, 2);
            if (!phase_barrier(a, 2, k)) return;
            if (PROF) tb = gtimer();
        }
        if (PROF && gtid == 0) {
            unsigned long long t = gtimer();
            tacc[1] += t - t0;
            if ((int64_t)k < a.nk_cap) a.rstat[16 * k + 5] = (int64_t)(t - t0);
            t0 = t;
        }
        // ------------------------------------------------------------ P3
        const unsigned long long ncol = cs[cI];
        const unsigned long long nqs = cs[cNQS], nq = cs[cNQ];
        // short rows: 4 rows per warp, 8 lanes per row, 4 entries per lane
        for (unsigned long long base = gwarp * 4; base < nqs; base += nwarps * 4) {
            const unsigned long long idx = base + (lane >> 3);
            uint32_t u = kNone;
            int64_t rs = 0, re = 0;
            if (idx < nqs) {
                u = a.NQS[idx];
                rs = a.ro[u];
                re = a.ro[u + 1];
                if ((lane & 7) == 0) atomicAnd(&a.M[u >> 5], ~(1u << (u & 31)));  // coloured now
            }
            notify_entries<4>(a, u, rs + (lane & 7), re, 8, k, Dout, dcount);
            if (PROF && (lane & 7) == 0) nvisN += (uint32_t)(re - rs);
        }
        // long rows: one kNotifySeg-entry segment per warp
        for (unsigned long long it = gwarp; it < nq; it += nwarps) {
            const long long cn0 = PROF ? clock64() : 0;
            const uint2 item = a.NQ[it];
            const uint32_t u = item.x;
            if (item.y == 0 && lane == 0) atomicAnd(&a.M[u >> 5], ~(1u << (u & 31)));
            const int64_t rs = a.ro[u] + (int64_t)item.y * kNotifySeg;
            const int64_t re = min(a.ro[u + 1], rs + (int64_t)kNotifySeg);
            notify_entries<kNotifySeg / 32>(a, u, rs + lane, re, 32, k, Dout, dcount);
            if (PROF && lane == 0) nvisN += (uint32_t)(re - rs);
            if (PROF) prof_max(a, k, 3, clock64() - cn0);
        }
        if (PROF && gtid == 0 && (int64_t)k < a.nk_cap) {
            a.rstat[16 * k + 1] = (int64_t)ncol;
            a.rstat[16 * k + 2] = (int64_t)cs[cLS];
            a.rstat[16 * k + 3] = (int64_t)nq;
            a.rstat[16 * k + 7] = (int64_t)cs[cSQ];
        }
        rem -= ncol;
        stage_flush(a, cs, dcount, Dout, pslot ? pslot + 3 : nullptr, tb, 3);
        if (!phase_barrier(a, 3, k)) return;
        if (PROF && gtid == 0) {
            unsigned long long t = gtimer();
            tacc[2] += t - t0;
            if ((int64_t)k < a.nk_cap) a.rstat[16 * k + 6] = (int64_t)(t - t0);
            t0 = t;
        }
    }
    if (gtid == 0) {
        a.ctr[kRem] = rem;
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
    GC_CUDA_TRY(cudaFuncSetAttribute(k_event_persistent<PROF>,
                                     cudaFuncAttributeMaxDynamicSharedMemorySize, (int)kStageBytes));
    GC_CUDA_TRY(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k_event_persistent<PROF>,
                                                              kThreads, kStageBytes));
    if (per_sm < 1) {
        set_error("persistent event kernel cannot be resident");
        return GC_ERR_CUDA;
    }
    const int blocks = per_sm * g->sm_count;
    void *args[] = {&a};
    GC_CUDA_TRY(cudaLaunchCooperativeKernel((void *)k_event_persistent<PROF>, blocks, kThreads, args,
                                            kStageBytes, g->stream));
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
    GC_CUDA_TRY(cudaMemsetAsync(s.M, 0xFF, sizeof(uint32_t) * (size_t)((n + 31) / 32), g->stream));
    GC_CUDA_TRY(cudaMemsetAsync(s.ctr, 0, 64 * sizeof(unsigned long long), g->stream));
    const unsigned long long rem = (unsigned long long)n;
    GC_CUDA_TRY(cudaMemcpyAsync(s.ctr + kRem, &rem, sizeof(rem), cudaMemcpyHostToDevice, g->stream));
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
    a.M = s.M;
    a.D[0] = s.F[0];
    a.D[1] = s.F[1];
    a.WQ = s.hub;
    a.SQ = reinterpret_cast<uint2 *>(s.Q2);
    a.LS = reinterpret_cast<LongScan *>(s.LS);
    a.NQS = s.Q;
    a.NQ = reinterpret_cast<uint2 *>(s.Q3);
    a.ctr = s.ctr;
    a.nk = s.nk;
    a.rstat = s.rstat;
    a.nk_cap = s.nk_cap;
    a.n = n;
    a.key = p.keys.k[0];
    a.max_rounds = (uint32_t)max_rounds;
    a.nq_cap = a.sq_cap = (unsigned long long)(n + g->nnz / 128 + 1);
    a.ls_cap = (unsigned long long)n;
    const bool prof = p.prof && p.prof->on;
    // GC_PROFILE_HIST=<file>: with GC_PROFILE, append the op-latency
    // histograms of this colouring to <file> (tools/round_profile.py)
    const char *hist_path = prof ? std::getenv("GC_PROFILE_HIST") : nullptr;
    a.hist = nullptr;
    if (hist_path && hist_path[0]) {
        if (!s.hist) GC_CUDA_TRY(dmalloc(&s.hist, 8 * 32 * sizeof(unsigned long long)));
        GC_CUDA_TRY(cudaMemsetAsync(s.hist, 0, 8 * 32 * sizeof(unsigned long long), g->stream));
        a.hist = s.hist;
    }
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
        snprintf(buf, sizeof(buf), "internal consistency check %llu failed in round %llu (vertex %llu)",
                 h[kErr - kRem], h[kErr - kRem + 1], h[kErr - kRem + 2]);
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
        // phase split (globaltimer, block 0): stored in ms[1..3] as fractions
        const double ns1 = (double)h[kPhaseNs - kRem], ns2 = (double)h[kPhaseNs + 1 - kRem],
                     ns3 = (double)h[kPhaseNs + 2 - kRem];
        p.prof->ms[1] += ns1 / 1e6;
        p.prof->ms[2] += ns2 / 1e6;
        p.prof->ms[3] += ns3 / 1e6;
        const int64_t visE = (int64_t)h[kVisE - kRem], visS = (int64_t)h[kVisS - kRem],
                      visN = (int64_t)h[kVisN - kRem], sumD = (int64_t)h[kSumD - kRem];
        // algorithmic bytes of the whole persistent kernel: per
        // evaluated vertex 4 B (D entry, not in round 0) + 16 B row offsets +
        // 16 B witness state (not in round 0) + 16 B state or 8 B colour/list
        // write; 4 B per scanned entry; per coloured vertex 4 B list + 16 B
        // offsets; per notified entry 4 B column id + 4 B colour + 8 B witness
        // ids of the neighbour.
        const int64_t b = 4 * (sumD - n) + 16 * sumD + 16 * (sumD - n) + 16 * (sumD - n) + 8 * n +
                          4 * (visE + visS) + 20 * n + 16 * visN;
        p.prof->bytes[0] += b;
        p.prof->visits += visE + visS;
        if (a.hist) {
            unsigned long long hh[8 * 32];
            GC_CUDA_TRY(cudaMemcpy(hh, a.hist, sizeof(hh), cudaMemcpyDeviceToHost));
            if (FILE *f = std::fopen(hist_path, "a")) {
                std::fprintf(f, "{\"n\": %lld, \"rounds\": %lld, \"hist\": [", (long long)n,
                             (long long)r->rounds);
                for (int i = 0; i < 8 * 32; ++i) std::fprintf(f, "%s%llu", i ? ", " : "", hh[i]);
                std::fprintf(f, "]}\n");
                std::fclose(f);
            }
        }
    }
    return GC_OK;
}

}  // namespace gc
