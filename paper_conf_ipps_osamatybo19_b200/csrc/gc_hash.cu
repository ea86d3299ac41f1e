// gc_hash.cu -- the paper's Hash IS colouring (Alg.6, P:L478-505, P:L557-614;
// SURVEY N2) made deterministic by readings R16-R20.
//
// Round k over the frontier F_k (vertices uncoloured at the round's start),
// five launches, every test reading the round-start state:
//   k_hash_propose  8-lane group per v: mx(v) / mn(v) = heaviest / lightest of
//                   {v} u (adj(v) n U_k) (R16); atomicOr of a max / min bit
//                   into prop[mx] / prop[mn] (OR: order-free, so deterministic)
//   k_hash_tent     thread per w: a proposed w takes the smallest used colour
//                   not in its prohibited table (Alg.6 L20-24, R17), else the
//                   new colour 2k (max-proposed) / 2k+1 (min only); a vertex
//                   flagged by an earlier old-colour conflict takes the new
//                   colour directly (R19)
//   k_hash_resolve  8-lane group per tentatively coloured w: reset if an old
//                   neighbour has its colour (code 2, sets the R19 flag) or a
//                   heavier uncoloured neighbour has the same tentative colour
//                   (code 1) (R18)
//   k_hash_commit   thread per w: survivors write C[w], their round and the
//                   used-colour bit; the rest are appended to F_{k+1}
//   k_hash_table    8-lane group per v in F_{k+1}: insert the colours of the
//                   neighbours coloured in round k, ascending, distinct, until
//                   the table holds T (R20)
// Frontier sizes live in device memory, so rounds are enqueued in batches
// and the host reads the size once per batch (empty rounds are no-ops).
#include <algorithm>

#include "gc_internal.cuh"

namespace gc {
namespace {

constexpr int kGroup = 8;  // lanes per vertex in the row-scanning kernels
constexpr int kThreads = 256;
constexpr uint32_t kNone = 0xFFFFFFFFu;
constexpr int64_t kLongMin = 512;  // rows longer than this go to a CTA (the *_long kernels)
constexpr int kLongThreads = 512;
constexpr int kTabOnePass = 8;  // table insertions done in one row pass (else repeated passes)

struct HashArgs {
    const int64_t *ro;
    const uint32_t *ci;
    uint32_t *C;
    uint32_t *prop;   // bit 0: proposed as a max, bit 1: as a min
    uint32_t *tent;   // tentative colour or kNone
    uint8_t *res;     // resolve code: 0 keep, 1 new-new collision, 2 old colour
    uint8_t *fresh;   // R19: must take a new colour
    uint32_t *rnd;    // round in which the vertex was coloured (kNone before)
    uint32_t *tab;    // T prohibited colours per vertex
    uint8_t *tlen;    // entries used
    uint32_t *used;   // bitmask of colours used so far
    uint32_t *wmx;    // last computed mx(v) / mn(v): still exact while uncoloured,
    uint32_t *wmn;    // since U only shrinks (the max of a subset that keeps it)
    unsigned long long *ctr;  // [0], [1]: frontier sizes; [2]: rounds run; [3..8] PROF;
                              // [10 + c]: long rows of class c this round
    uint32_t *longl[3];       // long rows deferred by class c (0 propose, 1 resolve, 2 table)
    uint32_t key;
    int T;
};

__device__ __forceinline__ uint32_t prio(const HashArgs &a, uint32_t v) { return weight_mix(v ^ a.key); }

// The lanes of one vertex's group (groups of a warp diverge independently).
__device__ __forceinline__ unsigned group_mask() {
    return ((1u << kGroup) - 1u) << ((threadIdx.x & 31) & ~(kGroup - 1));
}

__device__ __forceinline__ unsigned long long group_max(unsigned long long x) {
    const unsigned m = group_mask();
#pragma unroll
    for (int o = kGroup / 2; o > 0; o >>= 1) {
        unsigned long long y = __shfl_xor_sync(m, x, o, kGroup);
        x = y > x ? y : x;
    }
    return x;
}
__device__ __forceinline__ unsigned long long group_min(unsigned long long x) {
    const unsigned m = group_mask();
#pragma unroll
    for (int o = kGroup / 2; o > 0; o >>= 1) {
        unsigned long long y = __shfl_xor_sync(m, x, o, kGroup);
        x = y < x ? y : x;
    }
    return x;
}

__device__ __forceinline__ void push_long(const HashArgs &a, int c, uint32_t v) {
    const unsigned long long i = atomicAdd(&a.ctr[10 + c], 1ull);
    a.longl[c][i] = v;
}

// Block-wide max / min of a 64-bit key, result in every thread.
template <bool MAX>
__device__ __forceinline__ unsigned long long block_reduce(unsigned long long x) {
    __shared__ unsigned long long sm[kLongThreads / 32];
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) {
        unsigned long long y = __shfl_xor_sync(0xFFFFFFFFu, x, o);
        x = MAX ? (y > x ? y : x) : (y < x ? y : x);
    }
    __syncthreads();  // sm reused across calls
    if ((threadIdx.x & 31) == 0) sm[threadIdx.x >> 5] = x;
    __syncthreads();
    x = sm[0];
    for (int i = 1; i < (int)(blockDim.x >> 5); ++i) {
        const unsigned long long y = sm[i];
        x = MAX ? (y > x ? y : x) : (y < x ? y : x);
    }
    return x;
}

__global__ void k_hash_init(HashArgs a, uint32_t *F, int64_t n) {
    for (int64_t v = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; v < n;
         v += (int64_t)gridDim.x * blockDim.x) {
        a.C[v] = GC_UNC;
        a.prop[v] = 0;
        a.fresh[v] = 0;
        a.rnd[v] = kNone;
        a.tlen[v] = 0;
        a.wmx[v] = kNone;
        a.wmn[v] = kNone;
        F[v] = (uint32_t)v;
    }
}

// Alg.6 L8-18 with R16: the heaviest / lightest of {v} u (adj(v) n U_k).
// PROF: ctr[3 + 2c] += row entries scanned, ctr[4 + 2c] += rows scanned by
// row-scan class c (0 propose, 1 resolve, 2 table).
template <bool PROF>
__device__ __forceinline__ void prof_row(const HashArgs &a, int c, int lane, int64_t len) {
    if (PROF && lane == 0) {
        atomicAdd(&a.ctr[3 + 2 * c], (unsigned long long)len);
        atomicAdd(&a.ctr[4 + 2 * c], 1ull);
    }
}

template <bool PROF>
__global__ void k_hash_propose(HashArgs a, const uint32_t *__restrict__ F, int in) {
    const unsigned long long N = a.ctr[in];
    const int lane = threadIdx.x % kGroup;
    const int64_t groups = (int64_t)gridDim.x * (blockDim.x / kGroup);
    for (int64_t i = ((int64_t)blockIdx.x * blockDim.x + threadIdx.x) / kGroup; i < (int64_t)N;
         i += groups) {
        const uint32_t v = F[i];
        {
            // U_k is a subset of U_{k-1}: a cached argmax / argmin that is
            // still uncoloured is still the argmax / argmin (no rescan)
            const uint32_t cm = a.wmx[v], cn = a.wmn[v];
            if (cm != kNone && a.C[cm] == GC_UNC && a.C[cn] == GC_UNC) {
                if (lane == 0) {
                    atomicOr(&a.prop[cm], 1u);
                    atomicOr(&a.prop[cn], 2u);
                }
                continue;
            }
        }
        const int64_t e0 = a.ro[v], e1 = a.ro[v + 1];
        if (e1 - e0 > kLongMin) {
            if (lane == 0) push_long(a, 0, v);
            continue;
        }
        const unsigned long long self = ((unsigned long long)prio(a, v) << 32) | v;
        unsigned long long mx = self, mn = self;
        for (int64_t e = e0 + lane; e < e1; e += kGroup) {
            const uint32_t u = a.ci[e];
            if (a.C[u] != GC_UNC) continue;
            const unsigned long long key = ((unsigned long long)prio(a, u) << 32) | u;
            mx = key > mx ? key : mx;
            mn = key < mn ? key : mn;
        }
        prof_row<PROF>(a, 0, lane, e1 - e0);
        mx = group_max(mx);
        mn = group_min(mn);
        if (lane == 0) {
            atomicOr(&a.prop[(uint32_t)mx], 1u);
            atomicOr(&a.prop[(uint32_t)mn], 2u);
            a.wmx[v] = (uint32_t)mx;
            a.wmn[v] = (uint32_t)mn;
        }
    }
}

// Alg.6 L19-28 with R17 / R19.
__global__ void k_hash_tent(HashArgs a, const uint32_t *__restrict__ F, int in, uint32_t k) {
    const unsigned long long N = a.ctr[in];
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < (int64_t)N;
         i += (int64_t)gridDim.x * blockDim.x) {
        const uint32_t w = F[i];
        const uint32_t pr = a.prop[w];
        uint32_t t = kNone;
        if (pr) {
            a.prop[w] = 0;  // ready for the next round
            if (!a.fresh[w]) {
                const uint32_t *tw = a.tab + (size_t)w * a.T;
                const int len = a.tlen[w];
                const uint32_t words = (2 * k + 31) / 32;  // used colours are < 2k
                for (uint32_t wd = 0; wd < words && t == kNone; ++wd) {
                    uint32_t bits = a.used[wd];
                    while (bits) {
                        const uint32_t c = wd * 32 + (uint32_t)__ffs(bits) - 1;
                        bits &= bits - 1;
                        bool in_tab = false;
                        for (int j = 0; j < len; ++j) in_tab |= tw[j] == c;
                        if (!in_tab) {
                            t = c;
                            break;
                        }
                    }
                }
            }
            if (t == kNone) t = 2 * k + ((pr & 1u) ? 0u : 1u);
        }
        a.tent[w] = t;
    }
}

// P:L501-505 with R18 / R19.
template <bool PROF>
__global__ void k_hash_resolve(HashArgs a, const uint32_t *__restrict__ F, int in, uint32_t k) {
    const unsigned long long N = a.ctr[in];
    const int lane = threadIdx.x % kGroup;
    const int64_t groups = (int64_t)gridDim.x * (blockDim.x / kGroup);
    for (int64_t i = ((int64_t)blockIdx.x * blockDim.x + threadIdx.x) / kGroup; i < (int64_t)N;
         i += groups) {
        const uint32_t w = F[i];
        const uint32_t t = a.tent[w];
        if (t == kNone) continue;  // uniform over the group
        const int64_t e0 = a.ro[w], e1 = a.ro[w + 1];
        if (e1 - e0 > kLongMin) {
            if (lane == 0) push_long(a, 1, w);
            continue;
        }
        const uint32_t pw = prio(a, w);
        // an old neighbour can hold t only if t is not new (t < 2k) and the
        // table may have missed colours (it is full); otherwise the first
        // heavier collision decides (code 1), else the first old clash (2)
        const uint32_t stop = (t < 2 * k && a.tlen[w] >= a.T) ? 2u : 1u;
        const unsigned gm = group_mask();
        uint32_t code = 0;
        int64_t b = e0;
        for (; b < e1; b += kGroup) {
            const int64_t e = b + lane;
            if (e < e1) {
                const uint32_t u = a.ci[e];
                const uint32_t cu = a.C[u];
                if (cu != GC_UNC) {
                    if (cu == t) code = 2;
                } else if (a.tent[u] == t && prio(a, u) > pw) {
                    code = code > 1 ? code : 1;
                }
            }
            if (__any_sync(gm, code >= stop)) break;
        }
        prof_row<PROF>(a, 1, lane, (b + kGroup < e1 ? b + kGroup : e1) - e0);
        code = (uint32_t)group_max(code);
        if (lane == 0) a.res[w] = (uint8_t)code;
    }
}

__global__ void k_hash_commit(HashArgs a, const uint32_t *__restrict__ F, int in, uint32_t *Fout,
                              uint32_t k) {
    const unsigned long long N = a.ctr[in];
    if (blockIdx.x == 0 && threadIdx.x == 0 && N > 0) a.ctr[2] += 1;
    __shared__ unsigned s_cnt[kThreads / 32];
    __shared__ unsigned long long s_base;
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    for (int64_t i0 = (int64_t)blockIdx.x * blockDim.x; i0 < (int64_t)N; i0 += stride) {
        const int64_t i = i0 + threadIdx.x;
        bool keep_unc = false;
        uint32_t wv = 0;
        if (i < (int64_t)N) {
            const uint32_t w = F[i];
            const uint32_t t = a.tent[w];
            keep_unc = true;
            if (t != kNone) {
                const uint8_t r = a.res[w];
                if (r == 0) {
                    a.C[w] = t;
                    a.rnd[w] = k;
                    // a set bit never clears: skip the (same-address) atomic when
                    // it is already visible
                    if (!(*(volatile uint32_t *)&a.used[t >> 5] & (1u << (t & 31))))
                        atomicOr(&a.used[t >> 5], 1u << (t & 31));
                    keep_unc = false;
                } else if (r == 2) {
                    a.fresh[w] = 1;
                }
            }
            wv = w;
        }
        // block-aggregated append, one global atomic per block and step
        // (frontier order does not matter: every decision of a round is a
        // function of sets)
        const unsigned bal = __ballot_sync(0xFFFFFFFFu, keep_unc);
        const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
        if (lane == 0) s_cnt[warp] = __popc(bal);
        __syncthreads();
        if (threadIdx.x == 0) {
            unsigned tot = 0;
            for (int j = 0; j < (int)(blockDim.x >> 5); ++j) {
                const unsigned c = s_cnt[j];
                s_cnt[j] = tot;
                tot += c;
            }
            s_base = tot ? atomicAdd(&a.ctr[in ^ 1], (unsigned long long)tot) : 0ull;
        }
        __syncthreads();
        if (keep_unc) Fout[s_base + s_cnt[warp] + __popc(bal & ((1u << lane) - 1))] = wv;
        __syncthreads();  // s_cnt / s_base reused by the next step
    }
}

// P:L569-578 with R20: ascending insertion of the new neighbour colours.
template <bool PROF>
__global__ void k_hash_table(HashArgs a, const uint32_t *__restrict__ F, int in, uint32_t k) {
    const unsigned long long N = a.ctr[in];
    const int lane = threadIdx.x % kGroup;
    const int64_t groups = (int64_t)gridDim.x * (blockDim.x / kGroup);
    for (int64_t i = ((int64_t)blockIdx.x * blockDim.x + threadIdx.x) / kGroup; i < (int64_t)N;
         i += groups) {
        const uint32_t v = F[i];
        int len = a.tlen[v];
        if (len >= a.T) continue;
        uint32_t *tv = a.tab + (size_t)v * a.T;
        const int64_t e0 = a.ro[v], e1 = a.ro[v + 1];
        if (e1 - e0 > kLongMin) {
            if (lane == 0) push_long(a, 2, v);
            continue;
        }
        if (a.T - len <= kTabOnePass) {
            // one pass: every lane keeps its kTabOnePass smallest distinct new
            // colours that are not in the table (sorted, padded with kNone);
            // the group's smallest (T - len) are among their union
            uint32_t buf[kTabOnePass];
#pragma unroll
            for (int j = 0; j < kTabOnePass; ++j) buf[j] = kNone;
            for (int64_t e = e0 + lane; e < e1; e += kGroup) {
                const uint32_t u = a.ci[e];
                if (a.rnd[u] != k) continue;
                const uint32_t c = a.C[u];
                if (c >= buf[kTabOnePass - 1]) continue;
                bool dup = false;
#pragma unroll
                for (int j = 0; j < kTabOnePass; ++j) dup |= buf[j] == c;
                for (int j = 0; j < len; ++j) dup |= tv[j] == c;
                if (dup) continue;
                uint32_t cur = c;
#pragma unroll
                for (int j = 0; j < kTabOnePass; ++j) {  // sorted insert, drops the largest
                    const uint32_t lo = min(buf[j], cur), hi = max(buf[j], cur);
                    buf[j] = lo;
                    cur = hi;
                }
            }
            prof_row<PROF>(a, 2, lane, e1 - e0);
            const int need = a.T - len;
            for (int r = 0; r < need; ++r) {  // ascending merge of the lane lists
                const uint32_t m = (uint32_t)group_min(buf[0]);
                if (m == kNone) break;
                if (lane == 0) tv[len] = m;
                ++len;
                if (buf[0] == m) {
#pragma unroll
                    for (int j = 0; j + 1 < kTabOnePass; ++j) buf[j] = buf[j + 1];
                    buf[kTabOnePass - 1] = kNone;
                }
            }
            if (lane == 0) a.tlen[v] = (uint8_t)len;
            continue;
        }
        long long last = -1;
        while (len < a.T) {
            // the smallest colour > last among the neighbours coloured in round k
            unsigned long long best = ~0ull;
            for (int64_t e = e0 + lane; e < e1; e += kGroup) {
                const uint32_t u = a.ci[e];
                if (a.rnd[u] != k) continue;
                const unsigned long long c = a.C[u];
                if ((long long)c > last && c < best) best = c;
            }
            prof_row<PROF>(a, 2, lane, e1 - e0);
            best = group_min(best);
            if (best == ~0ull) break;
            last = (long long)best;
            bool in_tab = false;
            for (int j = 0; j < len; ++j) in_tab |= tv[j] == (uint32_t)best;
            if (!in_tab) {
                if (lane == 0) tv[len] = (uint32_t)best;
                ++len;
            }
        }
        if (lane == 0) a.tlen[v] = (uint8_t)len;
    }
}

// The rows deferred by the group kernels, one CTA per row (hubs of R-MAT).
template <bool PROF>
__global__ void __launch_bounds__(kLongThreads) k_hash_propose_long(HashArgs a) {
    const unsigned long long M = a.ctr[10];
    for (unsigned long long it = blockIdx.x; it < M; it += gridDim.x) {
        const uint32_t v = a.longl[0][it];
        const int64_t e0 = a.ro[v], e1 = a.ro[v + 1];
        const unsigned long long self = ((unsigned long long)prio(a, v) << 32) | v;
        unsigned long long mx = self, mn = self;
        for (int64_t e = e0 + threadIdx.x; e < e1; e += blockDim.x) {
            const uint32_t u = a.ci[e];
            if (a.C[u] != GC_UNC) continue;
            const unsigned long long key = ((unsigned long long)prio(a, u) << 32) | u;
            mx = key > mx ? key : mx;
            mn = key < mn ? key : mn;
        }
        prof_row<PROF>(a, 0, threadIdx.x, e1 - e0);
        mx = block_reduce<true>(mx);
        mn = block_reduce<false>(mn);
        if (threadIdx.x == 0) {
            atomicOr(&a.prop[(uint32_t)mx], 1u);
            atomicOr(&a.prop[(uint32_t)mn], 2u);
            a.wmx[v] = (uint32_t)mx;
            a.wmn[v] = (uint32_t)mn;
        }
    }
}

template <bool PROF>
__global__ void __launch_bounds__(kLongThreads) k_hash_resolve_long(HashArgs a, uint32_t k) {
    const unsigned long long M = a.ctr[11];
    for (unsigned long long it = blockIdx.x; it < M; it += gridDim.x) {
        const uint32_t w = a.longl[1][it];
        const uint32_t t = a.tent[w];
        const uint32_t pw = prio(a, w);
        const int64_t e0 = a.ro[w], e1 = a.ro[w + 1];
        const uint32_t stop = (t < 2 * k && a.tlen[w] >= a.T) ? 2u : 1u;  // as k_hash_resolve
        unsigned long long code = 0;
        int64_t b = e0;
        for (; b < e1; b += blockDim.x) {
            const int64_t e = b + threadIdx.x;
            if (e < e1) {
                const uint32_t u = a.ci[e];
                const uint32_t cu = a.C[u];
                if (cu != GC_UNC) {
                    if (cu == t) code = 2;
                } else if (a.tent[u] == t && prio(a, u) > pw) {
                    code = code > 1 ? code : 1;
                }
            }
            if (__syncthreads_or(code >= stop)) break;
        }
        prof_row<PROF>(a, 1, threadIdx.x, (b + (int64_t)blockDim.x < e1 ? b + blockDim.x : e1) - e0);
        code = block_reduce<true>(code);
        if (threadIdx.x == 0) a.res[w] = (uint8_t)code;
    }
}

template <bool PROF>
__global__ void __launch_bounds__(kLongThreads) k_hash_table_long(HashArgs a, uint32_t k) {
    const unsigned long long M = a.ctr[12];
    for (unsigned long long it = blockIdx.x; it < M; it += gridDim.x) {
        const uint32_t v = a.longl[2][it];
        int len = a.tlen[v];
        uint32_t *tv = a.tab + (size_t)v * a.T;
        const int64_t e0 = a.ro[v], e1 = a.ro[v + 1];
        long long last = -1;
        while (len < a.T) {  // uniform over the block
            unsigned long long best = ~0ull;
            for (int64_t e = e0 + threadIdx.x; e < e1; e += blockDim.x) {
                const uint32_t u = a.ci[e];
                if (a.rnd[u] != k) continue;
                const unsigned long long c = a.C[u];
                if ((long long)c > last && c < best) best = c;
            }
            prof_row<PROF>(a, 2, threadIdx.x, e1 - e0);
            best = block_reduce<false>(best);
            if (best == ~0ull) break;
            last = (long long)best;
            bool in_tab = false;
            for (int j = 0; j < len; ++j) in_tab |= tv[j] == (uint32_t)best;
            if (!in_tab) {
                __syncthreads();  // every thread has read tv[0..len) before it grows
                if (threadIdx.x == 0) tv[len] = (uint32_t)best;
                ++len;
            }
        }
        if (threadIdx.x == 0) a.tlen[v] = (uint8_t)len;
    }
}

}  // namespace

int run_hash_is(gc_graph *g, const RunParams &p, int T, RunResult *r) {
    NvtxRange nv_("Hash IS colouring");
    Scratch &s = g->s;
    const int64_t n = g->n;
    r->rounds = r->inner = r->launches = 0;
    if (n == 0) return GC_OK;
    if (n >= (1ll << 29)) {
        set_error("hash IS: colours 2k with k <= 2n + 2 must fit int32 (n < 2^29)");
        return GC_ERR_TOO_LARGE;
    }
    const size_t nn = (size_t)n;
    const size_t used_words = (4 * nn + 64) / 32 + 1;
    HashArgs a;
    a.ro = g->ro;
    a.ci = g->ci;
    a.C = s.C;
    a.key = p.keys.k[0];
    a.T = T;
    a.prop = a.tent = a.rnd = a.tab = a.used = nullptr;
    a.res = a.fresh = a.tlen = nullptr;
    a.ctr = nullptr;
    a.longl[0] = a.longl[1] = a.longl[2] = nullptr;
    a.wmx = a.wmn = nullptr;
    const size_t long_cap = (size_t)(g->nnz / kLongMin) + 1;
    int rc = GC_OK;
    cudaStream_t st = g->stream;
    const int grid = g->sm_count * 8;
    const int64_t max_rounds = 2 * n + 4;
    int64_t k = 0;
    int cur = 0;
    int batch = 4;
    const bool has_long = g->max_deg > kLongMin;
    const int grid_long = g->sm_count * 2;
    const bool prof = p.prof && p.prof->on;
    EventTimer tm;
    if (cudaSuccess != dmalloc(&a.prop, nn * 4) || cudaSuccess != dmalloc(&a.tent, nn * 4) ||
        cudaSuccess != dmalloc(&a.rnd, nn * 4) || cudaSuccess != dmalloc(&a.res, nn) ||
        cudaSuccess != dmalloc(&a.fresh, nn) || cudaSuccess != dmalloc(&a.tlen, nn) ||
        cudaSuccess != dmalloc(&a.tab, nn * (size_t)std::max(T, 1) * 4) ||
        cudaSuccess != dmalloc(&a.used, used_words * 4) || cudaSuccess != dmalloc(&a.ctr, 16 * 8) ||
        cudaSuccess != dmalloc(&a.wmx, nn * 4) || cudaSuccess != dmalloc(&a.wmn, nn * 4) ||
        cudaSuccess != dmalloc(&a.longl[0], long_cap * 4) ||
        cudaSuccess != dmalloc(&a.longl[1], long_cap * 4) ||
        cudaSuccess != dmalloc(&a.longl[2], long_cap * 4)) {
        rc = GC_ERR_OOM;
        set_error("hash IS: device allocation failed");
        goto out;
    }
    {
        cudaError_t e = cudaMemsetAsync(a.used, 0, used_words * 4, st);
        unsigned long long init[16] = {(unsigned long long)n};
        if (e == cudaSuccess) e = cudaMemcpyAsync(a.ctr, init, sizeof(init), cudaMemcpyHostToDevice, st);
        if (e == cudaSuccess) {
            k_hash_init<<<grid, kThreads, 0, st>>>(a, s.F[0], n);
            e = cudaGetLastError();
        }
        if (e == cudaSuccess) e = cudaStreamSynchronize(st);  // `init` is a stack buffer
        if (e != cudaSuccess) {
            rc = cuda_fail(e, "hash IS init");
            goto out;
        }
        r->launches += 1;
        for (;;) {
            for (int b = 0; b < batch; ++b, ++k) {
                const int in = cur;
                uint32_t *Fin = s.F[in], *Fout = s.F[in ^ 1];
                e = cudaMemsetAsync(a.ctr + (in ^ 1), 0, 8, st);
                if (e == cudaSuccess && has_long) e = cudaMemsetAsync(a.ctr + 10, 0, 3 * 8, st);
                if (e != cudaSuccess) break;
                if (prof) {
                    tm.begin(st, 0);
                    k_hash_propose<true><<<grid, kThreads, 0, st>>>(a, Fin, in);
                    if (has_long) k_hash_propose_long<true><<<grid_long, kLongThreads, 0, st>>>(a);
                    tm.end(st);
                    tm.begin(st, 3);
                    k_hash_tent<<<grid, kThreads, 0, st>>>(a, Fin, in, (uint32_t)k);
                    tm.end(st);
                    tm.begin(st, 1);
                    k_hash_resolve<true><<<grid, kThreads, 0, st>>>(a, Fin, in, (uint32_t)k);
                    if (has_long) k_hash_resolve_long<true><<<grid_long, kLongThreads, 0, st>>>(a, (uint32_t)k);
                    tm.end(st);
                    tm.begin(st, 3);
                    k_hash_commit<<<grid, kThreads, 0, st>>>(a, Fin, in, Fout, (uint32_t)k);
                    tm.end(st);
                    if (T > 0) {
                        tm.begin(st, 2);
                        k_hash_table<true><<<grid, kThreads, 0, st>>>(a, Fout, in ^ 1, (uint32_t)k);
                        if (has_long)
                            k_hash_table_long<true><<<grid_long, kLongThreads, 0, st>>>(a, (uint32_t)k);
                        tm.end(st);
                    }
                } else {
                    k_hash_propose<false><<<grid, kThreads, 0, st>>>(a, Fin, in);
                    if (has_long) k_hash_propose_long<false><<<grid_long, kLongThreads, 0, st>>>(a);
                    k_hash_tent<<<grid, kThreads, 0, st>>>(a, Fin, in, (uint32_t)k);
                    k_hash_resolve<false><<<grid, kThreads, 0, st>>>(a, Fin, in, (uint32_t)k);
                    if (has_long) k_hash_resolve_long<false><<<grid_long, kLongThreads, 0, st>>>(a, (uint32_t)k);
                    k_hash_commit<<<grid, kThreads, 0, st>>>(a, Fin, in, Fout, (uint32_t)k);
                    if (T > 0) {
                        k_hash_table<false><<<grid, kThreads, 0, st>>>(a, Fout, in ^ 1, (uint32_t)k);
                        if (has_long)
                            k_hash_table_long<false><<<grid_long, kLongThreads, 0, st>>>(a, (uint32_t)k);
                    }
                }
                r->launches += (T > 0 ? 5 : 4) + (has_long ? (T > 0 ? 3 : 2) : 0);
                cur ^= 1;
                e = cudaGetLastError();
                if (e != cudaSuccess) break;
            }
            if (e == cudaSuccess)
                e = cudaMemcpyAsync(s.host_pinned, a.ctr, 3 * 8, cudaMemcpyDeviceToHost, st);
            if (e == cudaSuccess) e = cudaStreamSynchronize(st);
            if (e != cudaSuccess) {
                rc = cuda_fail(e, "hash IS rounds");
                goto out;
            }
            if (prof && (rc = tm.drain(p.prof))) goto out;
            const unsigned long long left = (unsigned long long)s.host_pinned[cur];
            r->rounds = s.host_pinned[2];
            if (left == 0) break;
            if (k > max_rounds) {
                set_error("hash IS: round bound 2n + 4 passed (asymmetric adjacency?)");
                rc = GC_ERR_NOT_SYMMETRIC;
                goto out;
            }
            batch = std::min(batch * 2, 64);
        }
    }
    r->inner = r->rounds;
    if (prof) {
        // algorithmic bytes: a row scan reads the vertex id
        // (4 B) and its offsets (16 B) and 4 B of col_indices per entry
        // (status / weight gathers are L2-resident);
        // tent + commit read / write 24 B per frontier vertex
        unsigned long long c[16];
        GC_CUDA_TRY(cudaMemcpy(c, a.ctr, sizeof(c), cudaMemcpyDeviceToHost));
        int64_t frontier_sum = 0;
        for (int cl = 0; cl < 3; ++cl) {
            p.prof->bytes[cl] += 4 * (int64_t)c[3 + 2 * cl] + 20 * (int64_t)c[4 + 2 * cl];
            p.prof->visits += (int64_t)c[3 + 2 * cl];
        }
        frontier_sum = (int64_t)c[4];  // propose scans every frontier row once
        p.prof->bytes[3] += 24 * frontier_sum;
    }
out:
    // on an error path kernels may still be queued: the blocks go back to the
    // cache only when no pending work uses them (gc_alloc.cu contract)
    if (rc) cudaStreamSynchronize(st);
    dfree(a.prop);
    dfree(a.tent);
    dfree(a.rnd);
    dfree(a.res);
    dfree(a.fresh);
    dfree(a.tlen);
    dfree(a.tab);
    dfree(a.used);
    dfree(a.ctr);
    for (int c = 0; c < 3; ++c) dfree(a.longl[c]);
    dfree(a.wmx);
    dfree(a.wmn);
    return rc;
}

}  // namespace gc
