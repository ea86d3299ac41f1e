// gc_event_common.cuh -- device helpers of the event (witness/resume) mode,
// shared by the multi-kernel driver (gc_event.cu) and the persistent kernel
// (gc_persist.cu).  See the header comment of gc_event.cu for the method.
#pragma once

#include "gc_internal.cuh"

namespace gc {
namespace ev {

constexpr unsigned kFull = 0xFFFFFFFFu;
constexpr uint32_t kNone = 0xFFFFFFFFu;

__device__ __forceinline__ unsigned lane_id() { return threadIdx.x & 31u; }

struct Found {
    int64_t hpos = -1, lpos = -1;  // absolute edge index of the witness, -1 = none
    uint32_t hw = kNone, lw = kNone;
};

// Lane-serial witness search over [min(sh,sl), re).
__device__ __forceinline__ void lane_search(const uint32_t *__restrict__ ci, const uint32_t *C,
                                            uint32_t thresh, uint32_t key, uint32_t pv,
                                            bool need_hi, bool need_lo, int64_t sh, int64_t sl,
                                            int64_t re, Found &f, uint32_t &nvis) {
    int64_t s = need_hi ? sh : re;
    if (need_lo && sl < s) s = sl;
    for (int64_t e = s; e < re; ++e) {
        ++nvis;
        const uint32_t u = ci[e];
        if (C[u] < thresh) continue;  // coloured before round k
        const uint32_t pu = weight_mix(u ^ key);
        if (need_hi && f.hpos < 0 && e >= sh && pu > pv) {
            f.hpos = e;
            f.hw = u;
        }
        if (need_lo && f.lpos < 0 && e >= sl && pu < pv) {
            f.lpos = e;
            f.lw = u;
        }
        if ((!need_hi || f.hpos >= 0) && (!need_lo || f.lpos >= 0)) break;
    }
}

// Warp-cooperative witness search (all arguments warp-uniform).
__device__ __forceinline__ void warp_search(const uint32_t *__restrict__ ci, const uint32_t *C,
                                            uint32_t thresh, uint32_t key, uint32_t pv,
                                            bool need_hi, bool need_lo, int64_t sh, int64_t sl,
                                            int64_t re, Found &f, uint32_t &nvis) {
    const unsigned lane = lane_id();
    int64_t s = need_hi ? sh : re;
    if (need_lo && sl < s) s = sl;
    for (int64_t e0 = s; e0 < re; e0 += 64) {
        const int64_t e1 = e0 + lane, e2 = e0 + 32 + lane;
        const uint32_t u1 = e1 < re ? ci[e1] : 0u;
        const uint32_t u2 = e2 < re ? ci[e2] : 0u;
        const uint32_t c1 = e1 < re ? C[u1] : 0u;
        const uint32_t c2 = e2 < re ? C[u2] : 0u;
        nvis += (e1 < re) + (e2 < re);
        bool h1 = false, l1 = false, h2 = false, l2 = false;
        if (e1 < re && c1 >= thresh) {
            const uint32_t pu = weight_mix(u1 ^ key);
            h1 = need_hi && e1 >= sh && pu > pv;
            l1 = need_lo && e1 >= sl && pu < pv;
        }
        if (e2 < re && c2 >= thresh) {
            const uint32_t pu = weight_mix(u2 ^ key);
            h2 = need_hi && e2 >= sh && pu > pv;
            l2 = need_lo && e2 >= sl && pu < pv;
        }
        if (f.hpos < 0) {
            unsigned b1 = __ballot_sync(kFull, h1), b2 = __ballot_sync(kFull, h2);
            if (b1) {
                int l = __ffs(b1) - 1;
                f.hpos = e0 + l;
                f.hw = __shfl_sync(kFull, u1, l);
            } else if (b2) {
                int l = __ffs(b2) - 1;
                f.hpos = e0 + 32 + l;
                f.hw = __shfl_sync(kFull, u2, l);
            }
        }
        if (f.lpos < 0) {
            unsigned b1 = __ballot_sync(kFull, l1), b2 = __ballot_sync(kFull, l2);
            if (b1) {
                int l = __ffs(b1) - 1;
                f.lpos = e0 + l;
                f.lw = __shfl_sync(kFull, u1, l);
            } else if (b2) {
                int l = __ffs(b2) - 1;
                f.lpos = e0 + 32 + l;
                f.lw = __shfl_sync(kFull, u2, l);
            }
        }
        if ((!need_hi || f.hpos >= 0) && (!need_lo || f.lpos >= 0)) break;
    }
}

// Where a vertex of D_k resumes: which sides lost their witness and from where.
struct Resume {
    bool need_hi, need_lo;
    int64_t sh, sl;
};

__device__ __forceinline__ Resume resume_of(uint32_t v, int64_t rs, bool dense, const uint2 *W,
                                            const uint2 *P, const uint32_t *C, uint32_t thresh) {
    Resume r;
    if (dense) {
        r.need_hi = r.need_lo = true;
        r.sh = r.sl = rs;
    } else {
        const uint2 w = W[v];
        const uint2 p = P[v];
        r.need_hi = C[w.x] < thresh;  // hi witness coloured in an earlier round
        r.need_lo = C[w.y] < thresh;
        r.sh = rs + (int64_t)p.x + 1;
        r.sl = rs + (int64_t)p.y + 1;
    }
    return r;
}

// Commit v after its search: blocked -> store the new witnesses; otherwise
// colour (Alg.5 L37-42: min wins when both, R9).  Returns true if coloured.
__device__ __forceinline__ bool settle(uint32_t v, int64_t rs, const Resume &r, const Found &f,
                                       uint32_t k, uint32_t *C, uint2 *W, uint2 *P) {
    const bool has_hi = !r.need_hi || f.hpos >= 0;
    const bool has_lo = !r.need_lo || f.lpos >= 0;
    if (has_hi && has_lo) {
        if (r.need_hi && r.need_lo) {
            W[v] = make_uint2(f.hw, f.lw);
            P[v] = make_uint2((uint32_t)(f.hpos - rs), (uint32_t)(f.lpos - rs));
        } else if (r.need_hi) {
            W[v].x = f.hw;
            P[v].x = (uint32_t)(f.hpos - rs);
        } else {
            W[v].y = f.lw;
            P[v].y = (uint32_t)(f.lpos - rs);
        }
        return false;
    }
    C[v] = 2u * k + (has_lo ? 0u : 1u);  // atomic-free: single writer
    return true;
}

__device__ __forceinline__ void warp_append(bool pred, uint32_t v, uint32_t *list,
                                            unsigned long long *counter) {
    const unsigned m = __ballot_sync(kFull, pred);
    if (!m) return;
    const unsigned lane = lane_id();
    const unsigned leader = __ffs(m) - 1;
    unsigned long long base = 0;
    if (lane == leader) base = atomicAdd(counter, (unsigned long long)__popc(m));
    base = __shfl_sync(kFull, base, leader);
    if (pred) list[base + __popc(m & ((1u << lane) - 1u))] = v;
}

// Neighbour w of a vertex u coloured in round k must be re-evaluated in
// round k+1 iff it is uncoloured and u was one of its witnesses.  The stamp
// S[w] (round+1 of its last enqueue) removes duplicates (duplicate CSR entries,
// or both witnesses coloured in the same round).
__device__ __forceinline__ bool wake(uint32_t w, uint32_t u, uint32_t k, const uint32_t *C,
                                     const uint2 *W, uint32_t *S) {
    if (C[w] != GC_UNC) return false;
    const uint2 ww = W[w];
    if (ww.x != u && ww.y != u) return false;
    return atomicMax(&S[w], k + 1u) < k + 1u;
}

}  // namespace ev
}  // namespace gc
