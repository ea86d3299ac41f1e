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

enum : int { cSEnd = 0, cLo, cHi, cPairs, cLong, cErr, cErrV, cChunks, cTicket, kDCtrWords = 16 };

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
        GC_CUDA_TRY(dmalloc(&s.S, nl * 4));
        // long jobs of one round: own rows and ghost rows longer than kLongMin
        // (each at most nnz / kLongMin); chunk items: at most 2 nnz / kChunk + jobs
        s.L_cap = 2 * (p.nnz / kLongMin) + 16;
        s.LC_cap = 2 * (p.nnz / kChunk) + s.L_cap + 16;
        GC_CUDA_TRY(dmalloc(&s.L, (size_t)s.L_cap * sizeof(LongJob)));
        GC_CUDA_TRY(dmalloc(&s.LC, (size_t)s.LC_cap * sizeof(uint2)));
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
        GC_CUDA_TRY(cudaStreamSynchronize(st));
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
