// gc_dist_count.cu -- COUNT-mode max-min rounds on a graph
// partitioned by contiguous vertex ranges.
//
// Partition p owns rows [v0, v1) (global column ids), the hi/lo counts of its
// own vertices, and a replicated colour array C[n_global].  The counts of an
// owned vertex w drop when a neighbour is coloured: an owned neighbour's row
// walk decrements them directly; a REMOTE neighbour v is seen through the
// per-round exchange of coloured (v, colour) pairs and the partition's ghost
// rows (for every remote v, the owned vertices adjacent to v -- by symmetry
// the entries of v's row that point into the partition), walked once when v
// is coloured.  Round k on every partition:
//   1. colour the owned vertices scheduled for round k (2k+1 if the lo side
//      is free, R9; Alg.5 L37-42) and walk their rows (owned neighbours
//      only), publishing the pairs;
//   2. all-gather (pairs coloured, error flag) and the pairs themselves;
//   3. apply the remote pairs to C and walk their ghost rows.
// Every decrement of round k happens before round k+1 starts, so the
// scheduling (first freeing of a side, lo-freed-second stamps) is the
// single-GPU one and the colouring is identical for any partition.
#include <cub/cub.cuh>

#include <algorithm>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <vector>

#include "gc_dist.cuh"

namespace gc {

int fill_u32(uint32_t *p, uint32_t val, int64_t n, cudaStream_t st);

namespace {

constexpr unsigned kFull = 0xFFFFFFFFu;
constexpr uint32_t kLoF = 0x80000000u;     // S entry: scheduled by its lo side
constexpr uint32_t kNever = 0xFFFFFFFFu;
constexpr int64_t kLongMin = 256;          // rows (or ghost rows) longer: block chunks
constexpr int64_t kCountLongMin = 4096;    // counting pass: rows longer go to blocks
constexpr int64_t kChunk = 1024;
constexpr unsigned long long kDecHi = 0ull - (1ull << 32);
constexpr unsigned long long kDecLo = ~0ull;

enum : int { cSEnd = 0, cLo, cHi, cPairs, cLong, cErr, cErrV, cChunks, cTicket, kDCtrWords = 24 };

struct LongJob {
    int64_t s, e;     // entry range
    uint32_t v;       // global id of the walked vertex
    uint32_t ghost;   // 1: entries are owned ids (ghost row); 0: global ids (own row)
};

struct DCArgs {
    const int64_t *ro;
    const uint32_t *ci;
    const int64_t *goff;
    const uint32_t *gadj;
    uint32_t *C;
    unsigned long long *cnt;
    uint32_t *Z;
    uint32_t *S;
    LongJob *L;
    int64_t L_cap;
    uint2 *LC;         // chunk items (job, chunk) of the long jobs
    int64_t LC_cap;
    unsigned long long *ctr;
    uint2 *pairs;
    int64_t n_loc;
    uint32_t v0;
    uint32_t key;
    uint32_t k;
};

__device__ __forceinline__ unsigned lane_id() { return threadIdx.x & 31u; }

__device__ __forceinline__ void flag(const DCArgs &a, unsigned long long kind, uint32_t v) {
    if (atomicCAS(a.ctr + cErr, 0ull, kind) == 0ull) a.ctr[cErrV] = v;
}

// warp-aggregated append of `val` by the currently active lanes
__device__ __forceinline__ void push_s(const DCArgs &a, uint32_t val) {
    const unsigned m = __activemask();
    const int leader = __ffs(m) - 1;
    unsigned long long base = 0;
    if ((int)lane_id() == leader) base = atomicAdd(a.ctr + cSEnd, (unsigned long long)__popc(m));
    base = __shfl_sync(m, base, leader);
    const unsigned long long at = base + __popc(m & ((1u << lane_id()) - 1u));
    if (at < (unsigned long long)a.n_loc) a.S[at] = val;
    else flag(a, 2, val);
}

// a long row as a job + its kChunk-entry chunk items (so the block kernels
// grid-stride over chunks, whatever the mix of job lengths)
__device__ __forceinline__ void push_long(const DCArgs &a, int64_t s, int64_t e, uint32_t v, uint32_t ghost) {
    const unsigned long long i = atomicAdd(a.ctr + cLong, 1ull);
    const uint32_t nch = (uint32_t)((e - s + kChunk - 1) / kChunk);
    const unsigned long long b = atomicAdd(a.ctr + cChunks, (unsigned long long)nch);
    if ((int64_t)i >= a.L_cap || (int64_t)(b + nch) > a.LC_cap) {
        flag(a, 3, v);
        return;
    }
    a.L[i] = LongJob{s, e, v, ghost};
    for (uint32_t c = 0; c < nch; ++c) a.LC[b + c] = make_uint2((uint32_t)i, c);
}

// v (priority pv) is coloured in round k: decrement the side of owned w
// (local index lw, global id wg) that v belongs to; the first freeing of a
// side schedules w for round k+1; a lo side freed second stamps Z (R9).
__device__ __forceinline__ void dec(const DCArgs &a, uint32_t pv, uint32_t lw, uint32_t wg) {
    const bool hi = pv > weight_mix(wg ^ a.key);
    const unsigned long long old = atomicAdd(a.cnt + lw, hi ? kDecHi : kDecLo);
    const uint32_t side = hi ? (uint32_t)(old >> 32) : (uint32_t)old;
    const uint32_t other = hi ? (uint32_t)old : (uint32_t)(old >> 32);
    if (side == 1u) {
        if (other != 0u) push_s(a, lw | (hi ? 0u : kLoF));
        else if (!hi) a.Z[lw] = a.k + 1u;
    } else if (side == 0u) {
        flag(a, 4, wg);  // underflow: the adjacency multiset is not symmetric
    }
}

// entries [s, e) of an own row (global ids; remote ones skipped) or a ghost
// row (owned ids), lanes `sub` of `width`
template <bool GHOST>
__device__ __forceinline__ void walk_entries(const DCArgs &a, uint32_t pv, int64_t s, int64_t e,
                                             int64_t sub, int64_t width) {
    for (int64_t i = s + sub; i < e; i += width) {
        if (GHOST) {
            const uint32_t lw = a.gadj[i];
            dec(a, pv, lw, a.v0 + lw);
        } else {
            const uint32_t u = __ldcs(a.ci + i);
            const uint32_t lw = u - a.v0;
            if ((int64_t)lw < a.n_loc) dec(a, pv, lw, u);
        }
    }
}

// ---------------------------------------------------------------- counting
// hi / lo of every owned vertex: rows <= 16 a lane, <= kCountLongMin a warp,
// longer ones by blocks (k_dc_count_long + k_dc_count_fin); a zero side
// schedules the vertex for round 0.
__global__ void k_dc_count(DCArgs a) {
    const unsigned lane = lane_id();
    const int64_t gw = ((int64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const int64_t nw = ((int64_t)gridDim.x * blockDim.x) >> 5;
    for (int64_t base = gw * 32; base < a.n_loc; base += nw * 32) {
        const int64_t lv = base + lane;
        const bool valid = lv < a.n_loc;
        int64_t rs = 0, re = 0;
        if (valid) {
            rs = a.ro[lv];
            re = a.ro[lv + 1];
            a.Z[lv] = kNever;
        }
        const int64_t deg = re - rs;
        const uint32_t pv = weight_mix((a.v0 + (uint32_t)lv) ^ a.key);
        uint32_t h = 0;
        if (valid && deg <= 16) {
            for (int64_t e = rs; e < re; ++e) h += weight_mix(__ldcs(a.ci + e) ^ a.key) > pv ? 1u : 0u;
        }
        if (valid && deg > kCountLongMin) {
            a.cnt[lv] = 0ull;
            push_long(a, rs, re, a.v0 + (uint32_t)lv, 0u);
        }
        unsigned mid = __ballot_sync(kFull, valid && deg > 16 && deg <= kCountLongMin);
        while (mid) {
            const int src = __ffs(mid) - 1;
            mid &= mid - 1;
            const int64_t r0 = __shfl_sync(kFull, rs, src), r1 = __shfl_sync(kFull, re, src);
            const uint32_t p = __shfl_sync(kFull, pv, src);
            uint32_t hh = 0;
            for (int64_t e = r0 + lane; e < r1; e += 32) hh += weight_mix(__ldcs(a.ci + e) ^ a.key) > p ? 1u : 0u;
            hh = __reduce_add_sync(kFull, hh);
            if (lane == (unsigned)src) h = hh;
        }
        if (valid && deg <= kCountLongMin) {
            const uint32_t lo = (uint32_t)deg - h;
            a.cnt[lv] = ((unsigned long long)h << 32) | lo;
            if (h == 0u || lo == 0u) push_s(a, (uint32_t)lv | (lo == 0u ? kLoF : 0u));
        }
    }
}

__global__ void k_dc_count_long(DCArgs a) {
    __shared__ uint32_t red[32];
    const unsigned long long nc = a.ctr[cChunks];
    for (unsigned long long i = blockIdx.x; i < nc; i += gridDim.x) {
        const uint2 it = a.LC[i];
        const LongJob L = a.L[it.x];
        const uint32_t pv = weight_mix(L.v ^ a.key);
        const int64_t c0 = L.s + (int64_t)it.y * kChunk, c1 = min(L.e, c0 + kChunk);
        uint32_t h = 0;
        for (int64_t e = c0 + threadIdx.x; e < c1; e += blockDim.x)
            h += weight_mix(__ldcs(a.ci + e) ^ a.key) > pv ? 1u : 0u;
        h = __reduce_add_sync(kFull, h);
        if (lane_id() == 0) red[threadIdx.x >> 5] = h;
        __syncthreads();
        if (threadIdx.x == 0) {
            uint32_t t = 0;
            for (int w = 0; w < (int)(blockDim.x >> 5); ++w) t += red[w];
            const unsigned long long tot = (unsigned long long)(c1 - c0);
            atomicAdd(a.cnt + (L.v - a.v0), ((unsigned long long)t << 32) + (tot - t));
        }
        __syncthreads();
    }
}

__global__ void k_dc_count_fin(DCArgs a) {
    const unsigned long long nl = a.ctr[cLong];
    for (unsigned long long j = (unsigned long long)blockIdx.x * blockDim.x + threadIdx.x; j < nl;
         j += (unsigned long long)gridDim.x * blockDim.x) {
        const uint32_t lv = a.L[j].v - a.v0;
        const unsigned long long c = a.cnt[lv];
        const uint32_t hi = (uint32_t)(c >> 32), lo = (uint32_t)c;
        if (hi == 0u || lo == 0u) push_s(a, lv | (lo == 0u ? kLoF : 0u));
    }
}

// round bookkeeping: the next round's slice of S; clear the per-round counters
__device__ __forceinline__ void dc_advance(const DCArgs &a) {
    a.ctr[cLo] = a.ctr[cHi];
    a.ctr[cHi] = a.ctr[cSEnd];
    a.ctr[cPairs] = 0ull;
    a.ctr[cLong] = 0ull;
    a.ctr[cChunks] = 0ull;
}
__global__ void k_dc_advance(DCArgs a) { dc_advance(a); }

// whole block, end of a kernel: true in one thread of the block that finishes
// last (every block's writes and atomics are visible to it)
__device__ __forceinline__ bool last_block(const DCArgs &a) {
    __shared__ int last;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        last = atomicAdd(a.ctr + cTicket, 1ull) == gridDim.x - 1;
        if (last) {
            a.ctr[cTicket] = 0ull;
            __threadfence();
        }
    }
    __syncthreads();
    return threadIdx.x == 0 && last;
}

// ---------------------------------------------------------------- rounds
// 1. the owned vertices scheduled for round k: 8-lane groups
__global__ void k_dc_walk(DCArgs a, unsigned long long *cnt_send) {
    const unsigned lane = lane_id();
    const int64_t gid = ((int64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 3;
    const int64_t ng = ((int64_t)gridDim.x * blockDim.x) >> 3;
    const int64_t lo = (int64_t)a.ctr[cLo], hi = (int64_t)a.ctr[cHi];
    const int64_t sub = lane & 7u;
    for (int64_t i = lo + gid; i < hi; i += ng) {
        const uint32_t it = a.S[i];
        const uint32_t lv = it & ~kLoF;
        const uint32_t vg = a.v0 + lv;
        const int64_t rs = a.ro[lv], re = a.ro[lv + 1];
        if (sub == 0) {
            const bool lo_free = (it & kLoF) || a.Z[lv] <= a.k;
            const uint32_t c = 2u * a.k + (lo_free ? 1u : 0u);
            a.C[vg] = c;
            const unsigned long long at = atomicAdd(a.ctr + cPairs, 1ull);
            a.pairs[at] = make_uint2(vg, c);
            if (re - rs > kLongMin) push_long(a, rs, re, vg, 0u);
        }
        if (re - rs <= kLongMin) walk_entries<false>(a, weight_mix(vg ^ a.key), rs, re, sub, 8);
    }
    if (last_block(a)) {  // what the all-gather of this round sends: (pairs, error flag)
        cnt_send[0] = __ldcg(a.ctr + cPairs);
        cnt_send[1] = __ldcg(a.ctr + cErr);
    }
}

// 3. remote pairs: apply to C, walk the ghost rows (8-lane groups; long
// ghost rows as jobs)
__global__ void k_dc_ghost(DCArgs a, const uint2 *recv, const unsigned long long *cnt_recv, int world,
                           int self, int64_t stride) {
    const unsigned lane = lane_id();
    const int64_t gid = ((int64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 3;
    const int64_t ng = ((int64_t)gridDim.x * blockDim.x) >> 3;
    const int64_t sub = lane & 7u;
    int64_t off = 0;
    for (int r = 0; r < world; ++r) {
        const int64_t cnt = (int64_t)cnt_recv[2 * r];
        if (r == self) continue;
        const uint2 *src = recv + (int64_t)r * stride;
        for (int64_t i = gid; i < cnt; i += ng) {
            const uint2 pr = src[i];
            const int64_t gs = a.goff[pr.x], ge = a.goff[(int64_t)pr.x + 1];
            if (sub == 0) {
                a.C[pr.x] = pr.y;
                if (ge - gs > kLongMin) push_long(a, gs, ge, pr.x, 1u);
            }
            if (ge - gs <= kLongMin) walk_entries<true>(a, weight_mix(pr.x ^ a.key), gs, ge, sub, 8);
        }
        off += cnt;
    }
    (void)off;
}

// long rows / ghost rows of the round: blocks grid-stride over their chunks
__global__ void k_dc_long(DCArgs a) {
    const unsigned long long nc = a.ctr[cChunks];
    for (unsigned long long i = blockIdx.x; i < nc; i += gridDim.x) {
        const uint2 it = a.LC[i];
        const LongJob L = a.L[it.x];
        const uint32_t pv = weight_mix(L.v ^ a.key);
        const int64_t c0 = L.s + (int64_t)it.y * kChunk, c1 = min(L.e, c0 + kChunk);
        if (L.ghost) walk_entries<true>(a, pv, c0, c1, threadIdx.x, blockDim.x);
        else walk_entries<false>(a, pv, c0, c1, threadIdx.x, blockDim.x);
    }
    if (last_block(a)) dc_advance(a);  // the round is complete on this rank
}

// ------------------------------------------------ device-driven rounds
// One persistent cooperative launch per rank runs every round of the
// partitioned COUNT colouring; no host synchronisation and no
// per-round launch.  The blocks of the launch are split into one group per
// local partition (loopback: P partitions on one GPU; across GPUs: one per
// rank).  Round k of partition p:
//   A. its scheduled vertices S[lo, hi): colour (2k + lo-free, R9), PUSH the
//      pair (v, colour) into every other partition's inbox (peer memory
//      across GPUs: plain stores over NVLink), walk short own rows, queue
//      long ones;
//   B. group barrier; the group leader publishes (round tag, pairs, error)
//      in every other partition's mailbox with a system-scope release;
//   C. wait for every other partition's mailbox word of round k (acquire):
//      all pairs of the round are in p's inbox, and every partition now
//      holds the same totals (the termination / stall decisions agree);
//   D. apply the received pairs to C and walk their ghost rows, queue long
//      ones; group barrier; E. long rows and ghost rows by the whole group;
//      group barrier -- every decrement of round k precedes round k+1.
// Inbox and mailbox slots alternate with k % 2: a partition writes round
// k+2's pairs only after it has waited for round k+1's words, which p
// publishes after its own step D of round k.  Mailbox words carry the
// colouring epoch, so no clearing (and no host barrier) is needed between
// colourings.
constexpr int kMaxLocal = 8;     // local partitions per launch (loopback P <= 8)
constexpr int64_t kPLongMin = 32;  // rows / ghost rows longer: block chunks (one batch of kQ per thread)
constexpr int kMaxWorld = 64;
struct DPArgs {
    DCArgs part[kMaxLocal];
    Inbox box[kMaxWorld];
    int world, nlocal, first;
    uint32_t epoch;
    int64_t cap;
    int64_t n_global;
    unsigned long long *gbar;    // [kMaxLocal * 16] group barrier counters (monotone per launch)
    unsigned long long *res;     // [kMaxLocal * 16]: rounds, error, remaining (group leader writes)
    int64_t *nk;                 // frontier sizes N_k (first local partition)
    int64_t nk_cap;
    uint32_t max_rounds;
    int sys;                     // 1: partitions on other GPUs (system-scope fences), 0: one GPU
    unsigned long long *tl;      // GC_DIST_TIMELINE: per round 5 maxima (ns since the round top), or null
    int64_t tl_cap;
};
enum : int { cPairs2 = 10, cGChunks2 = 12, cChunks2 = 14 };  // [k % 2] per-round counters (DCState ctr)

__device__ __forceinline__ unsigned long long mbox_word(uint32_t epoch, uint32_t k, unsigned long long cnt,
                                                        unsigned long long err) {
    return ((unsigned long long)(epoch & 0xFFFFu) << 48) | ((unsigned long long)((k + 1u) & 0xFFFFu) << 32) |
           ((err & 3ull) << 30) | (cnt & 0x3FFFFFFFull);
}
__device__ __forceinline__ unsigned long long mbox_tag(uint32_t epoch, uint32_t k) {
    return mbox_word(epoch, k, 0, 0) >> 32;
}
__device__ __forceinline__ void st_release_sys(unsigned long long *p, unsigned long long v) {
    asm volatile("st.release.sys.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ unsigned long long ld_acquire_sys(const unsigned long long *p) {
    unsigned long long v;
    asm volatile("ld.acquire.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ void st_relaxed_sys(unsigned long long *p, unsigned long long v) {
    asm volatile("st.relaxed.sys.global.u64 [%0], %1;" ::"l"(p), "l"(v) : "memory");
}
__device__ __forceinline__ unsigned long long ld_relaxed_sys(const unsigned long long *p) {
    unsigned long long v;
    asm volatile("ld.relaxed.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ unsigned long long ld_acquire_gpu(const unsigned long long *p) {
    unsigned long long v;
    asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
    return v;
}
__device__ __forceinline__ unsigned long long gtimer_dp() {
    unsigned long long t;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
    return t;
}

// group barrier #epoch_no (monotone counter, release arrival / acquire spin);
// false after 4 s (the error is then recorded by the caller)
__device__ __forceinline__ bool group_barrier(unsigned long long *ctr, unsigned gsize, unsigned long long nbar) {
    __shared__ int ok_sh;
    __syncthreads();
    if (threadIdx.x == 0) {
        int ok = 1;
        asm volatile("red.release.gpu.global.add.u64 [%0], %1;" ::"l"(ctr), "l"(1ull) : "memory");
        const unsigned long long want = nbar * gsize, t0 = gtimer_dp();
        unsigned spins = 0;
        while (ld_acquire_gpu(ctr) < want) {
            if ((++spins & 255u) == 0u && gtimer_dp() - t0 > 4000000000ull) {
                ok = 0;
                break;
            }
        }
        ok_sh = ok;
    }
    __syncthreads();
    return ok_sh != 0;
}

// entries [s, e) of an own row (global ids; remote ones skipped) or a ghost
// row (owned ids), lanes `sub` of `width`; kQ entries per lane in flight (the
// atomics of a batch are issued together, not one round trip per entry)
constexpr int kQ = 4;
// device-driven rounds keep two scheduled lists, S[0, n_loc) and
// S[n_loc, 2 n_loc): a vertex freed in round k goes to list (k+1) % 2, whose
// length (ctr[cSL + (k+1) % 2]) is final at the round-end barrier and is not
// touched by round k+1's pushes -- every block reads the same round slice
// even when a fast block is already freeing round-(k+2) vertices
enum : int { cSL = 16 };  // [list] lengths (DCState ctr)
__device__ __forceinline__ void push_sk(const DCArgs &a, uint32_t val, uint32_t k) {
    const unsigned lst = (k + 1u) & 1u;
    const unsigned m = __activemask();
    const int leader = __ffs(m) - 1;
    unsigned long long base = 0;
    if ((int)lane_id() == leader) base = atomicAdd(a.ctr + cSL + lst, (unsigned long long)__popc(m));
    base = __shfl_sync(m, base, leader);
    const unsigned long long at = base + __popc(m & ((1u << lane_id()) - 1u));
    if (at < (unsigned long long)a.n_loc) a.S[(int64_t)lst * a.n_loc + (int64_t)at] = val;
    else flag(a, 2, val);
}
// skip (DESIGN 7.0, dead side): the parity of v's colour names a side of v
// that was free at the start of round k (odd: lo, all smaller neighbours are
// coloured; even: hi, all larger ones), so decrements to that side's
// neighbours are dead and not issued (skip 1: entries below v, 0: above)
template <bool GHOST>
__device__ __forceinline__ void walk_entries_k(const DCArgs &a, uint32_t pv, int64_t s, int64_t e, int64_t sub,
                                               int64_t width, uint32_t k, int skip) {
    for (int64_t i0 = s + sub; i0 < e; i0 += kQ * width) {
        uint32_t lw[kQ], wg[kQ];
        bool live[kQ];
#pragma unroll
        for (int q = 0; q < kQ; ++q) {
            const int64_t i = i0 + q * width;
            live[q] = i < e;
            if (GHOST) {
                lw[q] = live[q] ? a.gadj[i] : 0u;
                wg[q] = a.v0 + lw[q];
            } else {
                wg[q] = live[q] ? __ldcs(a.ci + i) : 0u;
                lw[q] = wg[q] - a.v0;
                live[q] = live[q] && (int64_t)lw[q] < a.n_loc;
            }
        }
        unsigned long long old[kQ];
        bool hi[kQ];
#pragma unroll
        for (int q = 0; q < kQ; ++q) {
            hi[q] = pv > weight_mix(wg[q] ^ a.key);
            live[q] = live[q] && hi[q] != (skip == 1);
            old[q] = live[q] ? atomicAdd(a.cnt + lw[q], hi[q] ? kDecHi : kDecLo) : 2ull;
        }
#pragma unroll
        for (int q = 0; q < kQ; ++q) {
            if (!live[q]) continue;
            const uint32_t side = hi[q] ? (uint32_t)(old[q] >> 32) : (uint32_t)old[q];
            const uint32_t other = hi[q] ? (uint32_t)old[q] : (uint32_t)(old[q] >> 32);
            if (side == 1u) {
                if (other != 0u) push_sk(a, lw[q] | (hi[q] ? 0u : kLoF), k);
                else if (!hi[q]) a.Z[lw[q]] = k + 1u;
            } else if (side == 0u) {
                flag(a, 4, wg[q]);
            }
        }
    }
}
// a self-contained chunk of a long row / ghost row (no job indirection in
// the round's critical chain): first entry, vertex, length | ghost flag
struct __align__(16) ChunkItem {
    int64_t c0;
    uint32_t v;
    uint32_t len;  // entries | kGhostBit
};
constexpr uint32_t kGhostBit = 0x80000000u;
__device__ __forceinline__ void push_long_k(const DCArgs &a, int64_t s, int64_t e, uint32_t v, uint32_t ghost,
                                            int par) {
    // own rows' chunks at [0, LC_cap), ghost rows' at [LC_cap, 2 LC_cap):
    // separate lists, so each is complete at its own group barrier
    const uint32_t nch = (uint32_t)((e - s + kChunk - 1) / kChunk);
    const unsigned long long b = atomicAdd(a.ctr + (ghost ? cGChunks2 : cChunks2) + par, (unsigned long long)nch);
    if ((int64_t)(b + nch) > a.LC_cap) {
        flag(a, 3, v);
        return;
    }
    ChunkItem *lc = reinterpret_cast<ChunkItem *>(a.LC) + (ghost ? a.LC_cap : 0);
    for (uint32_t c = 0; c < nch; ++c) {
        const int64_t c0 = s + (int64_t)c * kChunk;
        lc[b + c] = ChunkItem{c0, v, (uint32_t)min((int64_t)kChunk, e - c0) | (ghost ? kGhostBit : 0u)};
    }
}
// chunks [i0, i1) of the round's list, blocks of the group grid-stride
__device__ __forceinline__ void walk_chunks(const DCArgs &a, bool ghost, unsigned long long i0,
                                            unsigned long long i1, unsigned gb, unsigned gsize, uint32_t k) {
    const ChunkItem *lc = reinterpret_cast<const ChunkItem *>(a.LC) + (ghost ? a.LC_cap : 0);
    for (unsigned long long i = i0 + gb; i < i1; i += gsize) {
        const ChunkItem c = lc[i];
        const uint32_t pv = weight_mix(c.v ^ a.key);
        const int64_t c1 = c.c0 + (c.len & ~kGhostBit);
        const int skip = (int)(__ldcg(a.C + c.v) & 1u);  // (written before the group barrier)
        if (c.len & kGhostBit) walk_entries_k<true>(a, pv, c.c0, c1, threadIdx.x, blockDim.x, k, skip);
        else walk_entries_k<false>(a, pv, c.c0, c1, threadIdx.x, blockDim.x, k, skip);
    }
}

#ifndef GC_DC_THREADS
#define GC_DC_THREADS 256  // threads per block of the partitioned persistent kernel
#endif
#ifndef GC_DC_BPS
#define GC_DC_BPS 3        // its blocks per SM (at most; loopback s22 P=1/2/4/8: 2 -> 21.3/32.6/33.2/36.4 ms,
                           // 3 -> 20.9/31.7/31.7/33.0, 4 -> 21.6/32.4/31.8/31.7; 512 or 768 threads x 1: slower)
#endif
__global__ void __launch_bounds__(GC_DC_THREADS) k_dc_persistent(const __grid_constant__ DPArgs A) {
    const unsigned gsize = gridDim.x / (unsigned)A.nlocal;
    const unsigned lp = blockIdx.x / gsize;
    if (lp >= (unsigned)A.nlocal) return;  // blocks beyond the groups
    const unsigned gb = blockIdx.x - lp * gsize;
    const DCArgs &a = A.part[lp];
    const int p = A.first + (int)lp;
    const unsigned lane = lane_id();
    const int64_t gid = ((int64_t)gb * blockDim.x + threadIdx.x) >> 3;  // 8-lane group in the group
    const int64_t ng = ((int64_t)gsize * blockDim.x) >> 3;
    const int64_t sub = lane & 7u;
    unsigned long long *bar = A.gbar + 16 * lp;
    unsigned long long nbar = 0;
    __shared__ unsigned long long peer_cnt[kMaxWorld];
    __shared__ unsigned long long sh_tot, sh_err, sh_nrecv;
    int64_t remaining = A.n_global;
    // round 0: the counting pass's list S[cLo, cHi); round k >= 1: list k % 2
    int64_t lo = (int64_t)__ldcg(a.ctr + cLo), hi = (int64_t)__ldcg(a.ctr + cHi);
    uint32_t k = 0;
    unsigned long long err_out = 0;
    for (;; ++k) {
        const int par = (int)(k & 1u), npar = par ^ 1;
        const unsigned long long t_round = A.tl ? gtimer_dp() : 0ull;
        unsigned long long *tl = (A.tl && (int64_t)k < A.tl_cap && threadIdx.x == 0) ? A.tl + 8 * k : nullptr;
        if (gb == 0 && threadIdx.x == 0) {  // the next round's counters (last used in round k-1)
            a.ctr[cPairs2 + npar] = 0ull;
            a.ctr[cGChunks2 + npar] = 0ull;
            a.ctr[cChunks2 + npar] = 0ull;
            if (lp == 0 && (int64_t)k < A.nk_cap) A.nk[k] = remaining;
        }
        // A. own scheduled vertices
        for (int64_t i = lo + gid; i < hi; i += ng) {
            const uint32_t it = a.S[(k ? (int64_t)par * a.n_loc : 0) + i];
            const uint32_t lv = it & ~kLoF;
            const uint32_t vg = a.v0 + lv;
            const int64_t rs = a.ro[lv], re = a.ro[lv + 1];
            if (sub == 0) {
                const bool lo_free = (it & kLoF) || a.Z[lv] <= k;
                const uint32_t c = 2u * k + (lo_free ? 1u : 0u);
                a.C[vg] = c;
                const unsigned long long at = atomicAdd(a.ctr + cPairs2 + par, 1ull);
                if ((int64_t)at < A.cap) {
                    for (int q = 0; q < A.world; ++q)
                        if (q != p) A.box[q].recv[((int64_t)par * A.world + p) * A.cap + (int64_t)at] = make_uint2(vg, c);
                } else {
                    flag(a, 2, vg);
                }
                if (re - rs > kPLongMin) push_long_k(a, rs, re, vg, 0u, par);
            }
            if (re - rs <= kPLongMin)
                walk_entries_k<false>(a, weight_mix(vg ^ a.key), rs, re, sub, 8, k,
                                      ((it & kLoF) || a.Z[lv] <= k) ? 1 : 0);
        }
        // B. publish
        if (tl) atomicMax(tl + 0, gtimer_dp() - t_round);  // own walks done
        if (!group_barrier(bar, gsize, ++nbar)) { err_out = 5; break; }
        if (tl) atomicMax(tl + 1, gtimer_dp() - t_round);  // group barrier 1
        // the chunks of own long rows are all queued: walk them while the
        // other partitions' mailbox words are in flight (E1)
        const unsigned long long n_own = __ldcg(a.ctr + cChunks2 + par);
        const unsigned long long own = __ldcg(a.ctr + cPairs2 + par);
        // list par was consumed in A (all blocks passed barrier 1): reset its
        // length for round k+1's pushes (ordered before them by barrier 3)
        if (k && gb == 0 && threadIdx.x == 0) a.ctr[cSL + par] = 0ull;
        if (gb == 0 && threadIdx.x == 0 && A.world > 1) {
            const unsigned long long e = __ldcg(a.ctr + cErr) ? 1ull : 0ull;
            const unsigned long long w = mbox_word(A.epoch, k, own, e);
            // one system-scope fence, then the words (release pattern): the
            // pairs pushed by the whole group (ordered before the group
            // barrier this thread acquired) are visible before any word
            if (A.sys) asm volatile("fence.acq_rel.sys;" ::: "memory");
            else asm volatile("fence.acq_rel.gpu;" ::: "memory");
            for (int q = 0; q < A.world; ++q)
                if (q != p) st_relaxed_sys(A.box[q].mbox + (int64_t)par * A.world + p, w);
        }
        walk_chunks(a, false, 0, n_own, gb, gsize, k);
        // C. wait for every other partition's word of round k
        if (threadIdx.x < 32) {  // warp 0: lane q polls source q's word (all in flight together)
            const unsigned long long tag = mbox_tag(A.epoch, k), t0 = gtimer_dp();
            unsigned long long w = 0, c = 0, err = 0;
            bool done = false;
            unsigned spins = 0, bad = 0;
            for (;;) {
                bool mine = true;
                for (int q = (int)threadIdx.x; q < A.world; q += 32) {
                    if (q == p) continue;
                    w = ld_relaxed_sys(A.box[p].mbox + (int64_t)par * A.world + q);
                    mine = mine && (w >> 32) == tag;
                }
                done = __all_sync(0xFFFFFFFFu, mine);
                if (done) break;
                if ((++spins & 255u) == 0u && gtimer_dp() - t0 > 4000000000ull) {
                    bad = 1;
                    break;
                }
            }
            if (A.world > 1) {  // acquire pattern
                if (A.sys) asm volatile("fence.acq_rel.sys;" ::: "memory");
                else asm volatile("fence.acq_rel.gpu;" ::: "memory");
            }
            for (int q = (int)threadIdx.x; q < A.world; q += 32) {
                if (q == p) {
                    peer_cnt[q] = 0;
                    continue;
                }
                w = ld_relaxed_sys(A.box[p].mbox + (int64_t)par * A.world + q);
                peer_cnt[q] = w & 0x3FFFFFFFull;
                c += peer_cnt[q];
                err |= (w >> 30) & 3ull;
            }
            for (int o = 16; o; o >>= 1) {
                c += __shfl_xor_sync(0xFFFFFFFFu, c, o);
                err |= __shfl_xor_sync(0xFFFFFFFFu, err, o);
            }
            bad = __reduce_or_sync(0xFFFFFFFFu, bad);
            if (threadIdx.x == 0) {
                err |= __ldcg(a.ctr + cErr) ? 1ull : 0ull;
                sh_tot = own + c;
                sh_err = bad ? 6ull : (err ? 7ull : 0ull);
            }
        }
        __syncthreads();
        if (tl) atomicMax(tl + 2, gtimer_dp() - t_round);  // all mailboxes in
        const unsigned long long tot = sh_tot;
        if (sh_err) { err_out = sh_err; break; }  // an error on some partition: all stop (uniform)
        if (tot == 0) { err_out = 8; break; }     // a stall: the adjacency is not symmetric
        // D. remote pairs: C and ghost rows -- one index space over all
        // sources (peer_cnt holds the exclusive prefix after the scan below),
        // so every 8-lane group of the partition works at once
        if (threadIdx.x == 0) {
            unsigned long long acc = 0;
            for (int q = 0; q < A.world; ++q) {
                const unsigned long long c = peer_cnt[q];
                peer_cnt[q] = acc;
                acc += c;
            }
            sh_nrecv = acc;  // pairs received
        }
        __syncthreads();
        const int64_t nrecv = (int64_t)sh_nrecv;
        for (int64_t t = gid; t < nrecv; t += ng) {
            {
                int q = 0;
                while (q + 1 < A.world && (int64_t)peer_cnt[q + 1] <= t) ++q;
                const uint2 pr = A.box[p].recv[((int64_t)par * A.world + q) * A.cap + (t - (int64_t)peer_cnt[q])];
                const int64_t gs = a.goff[pr.x], ge = a.goff[(int64_t)pr.x + 1];
                if (sub == 0) {
                    a.C[pr.x] = pr.y;
                    if (ge - gs > kPLongMin) push_long_k(a, gs, ge, pr.x, 1u, par);
                }
                if (ge - gs <= kPLongMin)
                    walk_entries_k<true>(a, weight_mix(pr.x ^ a.key), gs, ge, sub, 8, k, (int)(pr.y & 1u));
            }
        }
        if (tl) atomicMax(tl + 3, gtimer_dp() - t_round);  // ghost walks done
        if (A.world > 1) {  // (one partition: no ghost rows, nothing queued here)
            if (!group_barrier(bar, gsize, ++nbar)) { err_out = 5; break; }
            if (tl) atomicMax(tl + 4, gtimer_dp() - t_round);  // group barrier 2
            // E2. the chunks of long ghost rows (queued after the own ones)
            walk_chunks(a, true, 0, __ldcg(a.ctr + cGChunks2 + par), gb, gsize, k);
        }
        if (tl) atomicMax(tl + 5, gtimer_dp() - t_round);  // long chunks done
        if (!group_barrier(bar, gsize, ++nbar)) { err_out = 5; break; }
        if (tl) atomicMax(tl + 6, gtimer_dp() - t_round);  // group barrier 3 (round end)
        remaining -= (int64_t)tot;
        lo = 0;
        hi = (int64_t)__ldcg(a.ctr + cSL + npar);
        if (remaining <= 0) {
            ++k;
            break;
        }
        if (k + 1 >= A.max_rounds) { err_out = 9; ++k; break; }
    }
    if (gb == 0 && threadIdx.x == 0) {
        A.res[16 * lp + 0] = k;
        A.res[16 * lp + 1] = err_out;
        A.res[16 * lp + 2] = (unsigned long long)remaining;
    }
}

// ---------------------------------------------------------------- ghost rows
__global__ void k_dc_gcount(const int64_t *ro, const uint32_t *ci, int64_t nnz, uint32_t v0, int64_t n_loc,
                            unsigned long long *gcnt) {
    for (int64_t e = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; e < nnz;
         e += (int64_t)gridDim.x * blockDim.x) {
        const uint32_t u = ci[e];
        if ((int64_t)(uint32_t)(u - v0) >= n_loc) atomicAdd(gcnt + (int64_t)u + 1, 1ull);
    }
}

__global__ void k_dc_gfill(const int64_t *ro, const uint32_t *ci, uint32_t v0, int64_t n_loc,
                           unsigned long long *cursor, uint32_t *gadj) {
    const unsigned lane = lane_id();
    const int64_t gw = ((int64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const int64_t nw = ((int64_t)gridDim.x * blockDim.x) >> 5;
    for (int64_t lv = gw; lv < n_loc; lv += nw) {
        for (int64_t e = ro[lv] + lane; e < ro[lv + 1]; e += 32) {
            const uint32_t u = ci[e];
            if ((int64_t)(uint32_t)(u - v0) >= n_loc) gadj[atomicAdd(cursor + u, 1ull)] = (uint32_t)lv;
        }
    }
}

int build_ghost(gc_graph *g, Part &p, int64_t n_global) {
    DCState &s = p.dc;
    const int64_t nl = p.v1 - p.v0;
    cudaStream_t st = g->stream;
    GC_CUDA_TRY(dmalloc(&s.goff, sizeof(int64_t) * (size_t)(n_global + 1)));
    GC_CUDA_TRY(cudaMemsetAsync(s.goff, 0, sizeof(int64_t) * (size_t)(n_global + 1), st));
    unsigned long long *g64 = reinterpret_cast<unsigned long long *>(s.goff);
    const int blocks = g->sm_count * 8;
    if (p.nnz > 0)
        k_dc_gcount<<<blocks, 256, 0, st>>>(p.ro, p.ci, p.nnz, (uint32_t)p.v0, nl, g64);
    size_t tmp_bytes = 0;
    GC_CUDA_TRY(cub::DeviceScan::InclusiveSum(nullptr, tmp_bytes, s.goff, s.goff, n_global + 1, st));
    void *tmp = nullptr;
    GC_CUDA_TRY(dmalloc(&tmp, std::max<size_t>(tmp_bytes, 16)));
    GC_CUDA_TRY(cub::DeviceScan::InclusiveSum(tmp, tmp_bytes, s.goff, s.goff, n_global + 1, st));
    int64_t ncut = 0;
    GC_CUDA_TRY(cudaMemcpyAsync(&ncut, s.goff + n_global, sizeof(int64_t), cudaMemcpyDeviceToHost, st));
    GC_CUDA_TRY(cudaStreamSynchronize(st));
    dfree(tmp);
    GC_CUDA_TRY(dmalloc(&s.gadj, sizeof(uint32_t) * (size_t)std::max<int64_t>(ncut, 1)));
    unsigned long long *cursor = nullptr;
    GC_CUDA_TRY(dmalloc(&cursor, sizeof(int64_t) * (size_t)(n_global + 1)));
    GC_CUDA_TRY(cudaMemcpyAsync(cursor, s.goff, sizeof(int64_t) * (size_t)(n_global + 1),
                                cudaMemcpyDeviceToDevice, st));
    if (nl > 0) k_dc_gfill<<<blocks, 256, 0, st>>>(p.ro, p.ci, (uint32_t)p.v0, nl, cursor, s.gadj);
    GC_CUDA_TRY(cudaGetLastError());
    GC_CUDA_TRY(cudaStreamSynchronize(st));
    dfree(cursor);
    s.ghost_built = true;
    return GC_OK;
}

int ensure_dc(gc_graph *g, Part &p, int64_t n_global) {
    DCState &s = p.dc;
    const size_t nl = (size_t)std::max<int64_t>(p.v1 - p.v0, 1);
    if (!s.cnt) {
        GC_CUDA_TRY(dmalloc(&s.cnt, nl * 8));
        GC_CUDA_TRY(dmalloc(&s.Z, nl * 4));
        GC_CUDA_TRY(dmalloc(&s.S, 2 * nl * 4));  // two lists (device-driven rounds)
        // long jobs of one round: own rows and ghost rows longer than kLongMin
        // (each at most nnz / kLongMin); chunk items: at most 2 nnz / kChunk + jobs
        s.L_cap = 2 * (p.nnz / std::min(kLongMin, kPLongMin)) + 16;  // own + ghost rows longer than the threshold
        s.LC_cap = 2 * (p.nnz / kChunk) + s.L_cap + 16;
        GC_CUDA_TRY(dmalloc(&s.L, (size_t)s.L_cap * sizeof(LongJob)));
        GC_CUDA_TRY(dmalloc(&s.LC, (size_t)s.LC_cap * 32));  // uint2 items (host rounds) or 2 lists of 16 B ChunkItems
        GC_CUDA_TRY(dmalloc(&s.ctr, kDCtrWords * sizeof(unsigned long long)));
    }
    if (!s.ghost_built) return build_ghost(g, p, n_global);
    return GC_OK;
}

DCArgs args_of(gc_graph *g, Part &p, uint32_t key, uint32_t k) {
    DCArgs a;
    a.ro = p.ro;
    a.ci = p.ci;
    a.goff = p.dc.goff;
    a.gadj = p.dc.gadj;
    a.C = p.C;
    a.cnt = p.dc.cnt;
    a.Z = p.dc.Z;
    a.S = p.dc.S;
    a.L = reinterpret_cast<LongJob *>(p.dc.L);
    a.L_cap = p.dc.L_cap;
    a.LC = reinterpret_cast<uint2 *>(p.dc.LC);
    a.LC_cap = p.dc.LC_cap;
    a.ctr = p.dc.ctr;
    a.pairs = p.colored;
    a.n_loc = p.v1 - p.v0;
    a.v0 = (uint32_t)p.v0;
    a.key = key;
    a.k = k;
    (void)g;
    return a;
}

}  // namespace

void free_dist_count(Part &p) {
    DCState &s = p.dc;
    dfree(s.cnt);
    dfree(s.Z);
    dfree(s.S);
    dfree(s.L);
    dfree(s.LC);
    dfree(s.goff);
    dfree(s.gadj);
    dfree(s.ctr);
    s = DCState();
}


// ------------------------------------------------ device-driven rounds: host
namespace {

// Inboxes of every partition.  One GPU (loopback): device allocations.  Across
// GPUs: each rank cudaMallocs its inbox, the IPC handles are all-gathered over
// the rank's NCCL communicator and the peers' inboxes are opened (NVLink peer
// access); any failure leaves the handle on the host-driven rounds.
int ensure_inboxes(gc_graph *g) {
    Dist &d = *g->dist;
    if (d.persist_state != 0) return GC_OK;
    const size_t recv_bytes = sizeof(uint2) * 2 * (size_t)d.world * (size_t)std::max<int64_t>(d.cap, 1);
    const size_t mbox_bytes = sizeof(unsigned long long) * 2 * (size_t)d.world;
    d.inbox.assign((size_t)d.world, Inbox());
    if (d.loopback) {
        for (int q = 0; q < d.world; ++q) {
            GC_CUDA_TRY(dmalloc(&d.inbox[q].recv, recv_bytes));
            GC_CUDA_TRY(dmalloc(&d.inbox[q].mbox, mbox_bytes));
            GC_CUDA_TRY(cudaMemsetAsync(d.inbox[q].mbox, 0, mbox_bytes, g->stream));
        }
        d.persist_state = 1;
        return GC_OK;
    }
#ifdef GC_HAVE_NCCL
    d.persist_state = -1;  // until every step below succeeded
    if (cudaMalloc(&d.own_recv, recv_bytes) != cudaSuccess || cudaMalloc(&d.own_mbox, mbox_bytes) != cudaSuccess) {
        cudaGetLastError();
        return GC_OK;
    }
    GC_CUDA_TRY(cudaMemsetAsync(d.own_mbox, 0, mbox_bytes, g->stream));
    cudaIpcMemHandle_t mine[2];
    if (cudaIpcGetMemHandle(&mine[0], d.own_recv) != cudaSuccess ||
        cudaIpcGetMemHandle(&mine[1], d.own_mbox) != cudaSuccess) {
        cudaGetLastError();
        return GC_OK;
    }
    char *dev = nullptr;
    const size_t hb = sizeof(mine);
    GC_CUDA_TRY(dmalloc(&dev, hb * (size_t)(d.world + 1)));
    GC_CUDA_TRY(cudaMemcpyAsync(dev + hb * (size_t)d.world, mine, hb, cudaMemcpyHostToDevice, g->stream));
    ncclResult_t ne = ncclAllGather(dev + hb * (size_t)d.world, dev, hb, ncclUint8, d.comm, g->stream);
    if (ne != ncclSuccess) {
        dfree(dev);
        return nccl_fail(ne, "ncclAllGather (inbox handles)");
    }
    std::vector<cudaIpcMemHandle_t> all(2 * (size_t)d.world);
    GC_CUDA_TRY(cudaMemcpyAsync(all.data(), dev, hb * (size_t)d.world, cudaMemcpyDeviceToHost, g->stream));
    if (int rw = dist_wait(g)) {
        dfree(dev);
        return rw;
    }
    dfree(dev);
    bool ok = true;
    for (int q = 0; q < d.world && ok; ++q) {
        if (q == d.rank) {
            d.inbox[q].recv = reinterpret_cast<uint2 *>(d.own_recv);
            d.inbox[q].mbox = reinterpret_cast<unsigned long long *>(d.own_mbox);
            continue;
        }
        void *pr = nullptr, *pm = nullptr;
        if (cudaIpcOpenMemHandle(&pr, all[2 * q], cudaIpcMemLazyEnablePeerAccess) != cudaSuccess) ok = false;
        else d.ipc_opened.push_back(pr);
        if (ok && cudaIpcOpenMemHandle(&pm, all[2 * q + 1], cudaIpcMemLazyEnablePeerAccess) != cudaSuccess) ok = false;
        else if (ok) d.ipc_opened.push_back(pm);
        d.inbox[q].recv = reinterpret_cast<uint2 *>(pr);
        d.inbox[q].mbox = reinterpret_cast<unsigned long long *>(pm);
    }
    cudaGetLastError();
    // every rank must agree (a rank without peer access makes all use host rounds)
    int *flag_d = nullptr;
    int flag_h = ok ? 1 : 0;
    GC_CUDA_TRY(dmalloc(&flag_d, sizeof(int)));
    GC_CUDA_TRY(cudaMemcpyAsync(flag_d, &flag_h, sizeof(int), cudaMemcpyHostToDevice, g->stream));
    ne = ncclAllReduce(flag_d, flag_d, 1, ncclInt32, ncclMin, d.comm, g->stream);
    if (ne == ncclSuccess) GC_CUDA_TRY(cudaMemcpyAsync(&flag_h, flag_d, sizeof(int), cudaMemcpyDeviceToHost, g->stream));
    if (int rw = dist_wait(g)) {
        dfree(flag_d);
        return rw;
    }
    dfree(flag_d);
    if (ne != ncclSuccess) return nccl_fail(ne, "ncclAllReduce (peer access)");
    d.persist_state = flag_h ? 1 : -1;
    return GC_OK;
#else
    d.persist_state = -1;
    return GC_OK;
#endif
}

bool use_persistent(gc_graph *g) {
    Dist &d = *g->dist;
    const char *e = std::getenv("GC_DIST_HOST_ROUNDS");  // A/B: the host-driven rounds
    if (e && e[0] == '1') return false;
    if ((int)d.parts.size() > kMaxLocal || d.world > kMaxWorld) return false;
    if (ensure_inboxes(g) != GC_OK) return false;
    return d.persist_state == 1;
}

int run_dist_persistent(gc_graph *g, const RunParams &p, RunResult *r, int64_t *frontier, int64_t fcap) {
    NvtxRange nv_("partitioned COUNT rounds (device-driven)");
    Dist &d = *g->dist;
    cudaStream_t st = g->stream;
    const int nlocal = (int)d.parts.size();
    DPArgs A;
    memset(&A, 0, sizeof(A));
    for (int lp = 0; lp < nlocal; ++lp) A.part[lp] = args_of(g, d.parts[lp], p.keys.k[0], 0);
    for (int q = 0; q < d.world; ++q) A.box[q] = d.inbox[q];
    A.world = d.world;
    A.nlocal = nlocal;
    A.first = d.loopback ? 0 : d.rank;
    A.epoch = ++d.epoch;
    A.cap = std::max<int64_t>(d.cap, 1);
    A.n_global = d.n_global;
    A.max_rounds = (uint32_t)std::min<int64_t>(p.max_rounds, 0xFFFFFFF0ll);
    A.sys = d.loopback ? 0 : 1;
    const char *tle = std::getenv("GC_DIST_TIMELINE");  // experiments: per-round phase timeline
    unsigned long long *tlbuf = nullptr;
    const int64_t tl_cap = tle ? 1 << 14 : 0;
    if (tl_cap) {
        GC_CUDA_TRY(dmalloc(&tlbuf, (size_t)tl_cap * 64));
        GC_CUDA_TRY(cudaMemsetAsync(tlbuf, 0, (size_t)tl_cap * 64, st));
    }
    A.tl = tlbuf;
    A.tl_cap = tl_cap;
    const int64_t nk_cap = std::min<int64_t>(fcap > 0 ? fcap : 0, 1 << 20);
    unsigned long long *scratch = nullptr;  // gbar [16 kMaxLocal] + res [16 kMaxLocal] + nk
    const size_t words = 32 * (size_t)kMaxLocal + (size_t)std::max<int64_t>(nk_cap, 1);
    GC_CUDA_TRY(dmalloc(&scratch, words * 8));
    GC_CUDA_TRY(cudaMemsetAsync(scratch, 0, 32 * (size_t)kMaxLocal * 8, st));
    A.gbar = scratch;
    A.res = scratch + 16 * kMaxLocal;
    A.nk = reinterpret_cast<int64_t *>(scratch + 32 * kMaxLocal);
    A.nk_cap = nk_cap;
    int per_sm = 0;
    GC_CUDA_TRY(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, k_dc_persistent, GC_DC_THREADS, 0));
    const int gsize = std::max(1, (std::min(per_sm, GC_DC_BPS) * g->sm_count) / nlocal);
    cudaLaunchAttribute attr;
    attr.id = cudaLaunchAttributeCooperative;
    attr.val.cooperative = 1;
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = dim3((unsigned)(gsize * nlocal));
    cfg.blockDim = dim3(GC_DC_THREADS);
    cfg.stream = st;
    cfg.attrs = &attr;
    cfg.numAttrs = 1;
    cudaError_t le = cudaLaunchKernelEx(&cfg, k_dc_persistent, A);
    if (le != cudaSuccess) {
        dfree(scratch);
        return cuda_fail(le, "k_dc_persistent launch");
    }
    r->launches += 1;
    unsigned long long res[16 * kMaxLocal];
    GC_CUDA_TRY(cudaMemcpyAsync(res, A.res, sizeof(res), cudaMemcpyDeviceToHost, st));
    std::vector<int64_t> nk((size_t)std::max<int64_t>(nk_cap, 1));
    if (nk_cap > 0) GC_CUDA_TRY(cudaMemcpyAsync(nk.data(), A.nk, 8 * (size_t)nk_cap, cudaMemcpyDeviceToHost, st));
    GC_CUDA_TRY(cudaStreamSynchronize(st));
    dfree(scratch);
    if (tl_cap) {  // mean over rounds 10.. of each phase end (us), to stderr
        std::vector<unsigned long long> t((size_t)tl_cap * 8);
        GC_CUDA_TRY(cudaMemcpy(t.data(), tlbuf, t.size() * 8, cudaMemcpyDeviceToHost));
        dfree(tlbuf);
        const int64_t R = std::min<int64_t>((int64_t)res[0], tl_cap);
        double sum[7] = {0};
        for (int64_t k = std::min<int64_t>(10, R); k < R; ++k)
            for (int c = 0; c < 7; ++c) sum[c] += (double)t[8 * k + c];
        const double cnt = (double)std::max<int64_t>(1, R - std::min<int64_t>(10, R));
        fprintf(stderr, "dist timeline (us, mean of rounds >= 10, max over blocks): own-walks %.2f bar1 %.2f mbox %.2f "
                "ghost %.2f bar2 %.2f long %.2f bar3 %.2f\n", sum[0] / cnt / 1e3, sum[1] / cnt / 1e3, sum[2] / cnt / 1e3,
                sum[3] / cnt / 1e3, sum[4] / cnt / 1e3, sum[5] / cnt / 1e3, sum[6] / cnt / 1e3);
    }
    unsigned long long err = 0, local_kind = 0;
    for (int lp = 0; lp < nlocal; ++lp) {
        err = std::max(err, res[16 * lp + 1]);
        unsigned long long c[kDCtrWords];
        GC_CUDA_TRY(cudaMemcpy(c, d.parts[lp].dc.ctr, sizeof(c), cudaMemcpyDeviceToHost));
        if (c[cErr]) local_kind = c[cErr];
    }
    if (err) {
        if (err == 5 || err == 6) {
            set_error("distributed COUNT rounds: a partition stopped answering (device-side timeout)");
            return d.loopback ? GC_ERR_CUDA : GC_ERR_NCCL;
        }
        if (err == 9) {
            set_error("distributed colouring exceeded the round limit");
            return GC_ERR_TOO_LARGE;
        }
        if (local_kind == 2 || local_kind == 3) {
            set_error("internal: distributed COUNT list overflow");
            return GC_ERR_CUDA;
        }
        set_error("distributed COUNT colouring: the adjacency is not symmetric");
        return GC_ERR_NOT_SYMMETRIC;
    }
    r->rounds = (int64_t)res[0];
    r->inner = r->rounds;
    for (int64_t k = 0; frontier && k < std::min<int64_t>(fcap, r->rounds) && k < nk_cap; ++k) frontier[k] = nk[k];
    return GC_OK;
}

}  // namespace

void free_inboxes(Dist &d) {
    if (d.loopback) {
        for (auto &b : d.inbox) {
            dfree(b.recv);
            dfree(b.mbox);
        }
    } else {
        for (void *ptr : d.ipc_opened) cudaIpcCloseMemHandle(ptr);
        if (d.own_recv) cudaFree(d.own_recv);
        if (d.own_mbox) cudaFree(d.own_mbox);
    }
    d.inbox.clear();
    d.ipc_opened.clear();
    d.own_recv = d.own_mbox = nullptr;
    d.persist_state = 0;
}

int run_dist_count(gc_graph *g, const RunParams &p, RunResult *r, int64_t *frontier, int64_t fcap) {
    Dist &d = *g->dist;
    const int64_t n = d.n_global;
    cudaStream_t st = g->stream;
    const uint32_t key = p.keys.k[0];
    r->rounds = r->inner = r->launches = 0;
    const int blocks = g->sm_count * 8;
    if (!g->deduped && !g->rows_strict) {
        // the counts need a symmetric adjacency MULTISET: duplicate entries
        // (legal input, R13) are removed from this rank's rows first -- the
        // same adjacency sets, so the same colouring on every rank
        int rc = ensure_strict_rows(g);
        if (rc) return rc;
        if (g->deduped && (rc = dist_reslice(g))) return rc;
    }
    for (auto &pt : d.parts) {
        int rc = ensure_dc(g, pt, n);
        if (rc) return rc;
    }
    // GC_PROFILE: class 0 = the whole round loop (counting pass included) on
    // this rank, its algorithmic bytes: 16 B per owned vertex (offsets + count
    // word) + 4 B per own entry for counting; per own entry walked 4 B id +
    // 16 B count RMW when the neighbour is owned; per ghost entry 4 B + 16 B;
    // 8 B per coloured pair sent, 8 B per pair received.
    const bool prof = p.prof && p.prof->on;
    cudaEvent_t pe0 = nullptr, pe1 = nullptr;
    if (prof) {
        GC_CUDA_TRY(cudaEventCreate(&pe0));
        GC_CUDA_TRY(cudaEventCreate(&pe1));
        GC_CUDA_TRY(cudaEventRecord(pe0, st));
    }
    for (auto &pt : d.parts) {
        int rc = GC_OK;
        rc = fill_u32(pt.C, GC_UNC, n, st);
        if (rc) return rc;
        GC_CUDA_TRY(cudaMemsetAsync(pt.dc.ctr, 0, kDCtrWords * sizeof(unsigned long long), st));
        DCArgs a = args_of(g, pt, key, 0);
        if (a.n_loc > 0) {
            k_dc_count<<<blocks, 256, 0, st>>>(a);
            k_dc_count_long<<<blocks, 256, 0, st>>>(a);
            k_dc_count_fin<<<g->sm_count, 256, 0, st>>>(a);
        }
        k_dc_advance<<<1, 1, 0, st>>>(a);
        r->launches += 4;
    }
    GC_CUDA_TRY(cudaGetLastError());
    if (use_persistent(g)) {
        int rc = run_dist_persistent(g, p, r, frontier, fcap);
        if (rc) return rc;
        if (prof) {
            GC_CUDA_TRY(cudaEventRecord(pe1, st));
            GC_CUDA_TRY(cudaEventSynchronize(pe1));
            float ms = 0.f;
            cudaEventElapsedTime(&ms, pe0, pe1);
            cudaEventDestroy(pe0);
            cudaEventDestroy(pe1);
            p.prof->ms[0] += ms;
            p.prof->launches[0] += 1;
            p.prof->launch_us.push_back(1e3f * ms);
        }
        return GC_OK;
    }
    std::vector<const void *> cs(d.parts.size()), ps(d.parts.size());
    std::vector<void *> cr(d.parts.size()), pr(d.parts.size());
    for (size_t q = 0; q < d.parts.size(); ++q) {
        cs[q] = d.parts[q].cnt_send;
        cr[q] = d.parts[q].cnt_recv;
        ps[q] = d.parts[q].colored;
        pr[q] = d.parts[q].recv;
    }
    int64_t remaining = n, k = 0;
    while (remaining > 0) {
        if (k >= p.max_rounds || k >= 0xFFFFFFF0ll) {
            set_error("distributed colouring exceeded the round limit");
            return GC_ERR_TOO_LARGE;
        }
        if (frontier && k < fcap) frontier[k] = remaining;
        for (auto &pt : d.parts) {
            DCArgs a = args_of(g, pt, key, (uint32_t)k);
            k_dc_walk<<<blocks, 256, 0, st>>>(a, pt.cnt_send);
            r->launches += 1;
        }
        int rc = dist_exchange(g, 2 * sizeof(unsigned long long), cs, cr);
        if (rc) return rc;
        GC_CUDA_TRY(cudaMemcpyAsync(d.host_cnt, d.parts[0].cnt_recv, 2 * sizeof(unsigned long long) * d.world,
                                    cudaMemcpyDeviceToHost, st));
        if ((rc = dist_wait(g))) return rc;
        unsigned long long maxc = 0, tot = 0, err = 0;
        for (int q = 0; q < d.world; ++q) {
            maxc = std::max(maxc, d.host_cnt[2 * q]);
            tot += d.host_cnt[2 * q];
            err |= d.host_cnt[2 * q + 1];
        }
        if (err || tot == 0) {
            // a count underflow or a stall: the adjacency (multiset) is not symmetric
            set_error(err == 2 || err == 3 ? "internal: distributed COUNT list overflow"
                                           : "distributed COUNT colouring: the adjacency is not symmetric");
            return (err == 2 || err == 3) ? GC_ERR_CUDA : GC_ERR_NOT_SYMMETRIC;
        }
        if (maxc > (unsigned long long)d.cap) {
            set_error("internal: coloured pairs exceed the partition capacity");
            return GC_ERR_CUDA;
        }
        rc = dist_exchange(g, sizeof(uint2) * maxc, ps, pr);
        if (rc) return rc;
        for (size_t q = 0; q < d.parts.size(); ++q) {
            Part &pt = d.parts[q];
            DCArgs a = args_of(g, pt, key, (uint32_t)k);
            const int self = d.loopback ? (int)q : d.rank;
            k_dc_ghost<<<blocks, 256, 0, st>>>(a, pt.recv, pt.cnt_recv, d.world, self, (int64_t)maxc);
            k_dc_long<<<blocks, 256, 0, st>>>(a);
            r->launches += 2;
        }
        GC_CUDA_TRY(cudaGetLastError());
        remaining -= (int64_t)tot;
        ++k;
    }
    r->rounds = k;
    r->inner = k;
    if (prof) {
        GC_CUDA_TRY(cudaEventRecord(pe1, st));
        GC_CUDA_TRY(cudaEventSynchronize(pe1));
        float ms = 0.f;
        cudaEventElapsedTime(&ms, pe0, pe1);
        cudaEventDestroy(pe0);
        cudaEventDestroy(pe1);
        int64_t bytes = 0, ents = 0;
        for (auto &pt : d.parts) {
            int64_t ncut = 0;
            GC_CUDA_TRY(cudaMemcpy(&ncut, pt.dc.goff + n, sizeof(int64_t), cudaMemcpyDeviceToHost));
            const int64_t nl = pt.v1 - pt.v0;
            bytes += 16 * nl + 4 * pt.nnz + 20 * pt.nnz + 20 * ncut + 8 * nl + 8 * n;
            ents += pt.nnz + ncut;
        }
        p.prof->ms[0] += ms;
        p.prof->launches[0] += 1;  // the round loop of one colouring (r->launches kernels)
        p.prof->bytes[0] += bytes;
        p.prof->visits += ents;
        p.prof->launch_us.push_back(1e3f * ms);
    }
    return GC_OK;
}

}  // namespace gc
