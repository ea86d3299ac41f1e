// gc_luby.cu -- Luby maximal-independent-set colouring on the GPU.
//
// Alg.2 outer loop "for each color" with the Alg.3 inner
// do-while that grows a maximal independent set:
//   phase A (Alg.3 L6-12): a candidate whose weight beats every candidate
//       neighbour joins the set (mis <- 1, weight <- 0);
//   phase B (Alg.3 L19-20): candidates adjacent to a new member drop out;
//   the do-while ends when no candidate is left; then Alg.2 L17 colours the
//   set and the remaining vertices restart as candidates with the SAME
//   weights (R10).
//
// State per vertex, S[v] (uint32): CAND = 0xFFFFFFFF; 2t = joined the set in
// inner iteration t; 2t+1 = dropped out in iteration t (t counts inner
// iterations over the whole run).  Phase A tests "S[u] == CAND || S[u] == 2t"
// so members joining concurrently in the same phase still count as
// candidates (the snapshot of Alg.3 L6), and vertices coloured earlier keep
// an old even stamp and never match.  Phase B tests "S[u] == 2t".
//
// The whole loop is driven from device memory: each inner iteration is three
// kernels (phase A, phase B, commit-if-done) that read the current list, the
// colour and the candidate count from a control block, so the host only
// checks for completion once per batch of iterations.
#include "gc_internal.cuh"

namespace gc {

namespace {

constexpr int kBlock = 256;
constexpr unsigned kFull = 0xFFFFFFFFu;
constexpr uint32_t kCand = 0xFFFFFFFFu;

// control block in g->s.ctr
enum : int {
    kCur = 8,        // which list buffer (0/1) holds the uncoloured list
    kLen = 9,        // its length
    kColor = 10,     // current colour c (0-based)
    kCandLeft = 11,  // candidates left after phase B
    kNextLen = 12,   // commit: length of the next list
    kTicket = 13,    // commit: last-block detection
    kBusy = 15       // inner iterations with a non-empty candidate set
};

__device__ __forceinline__ unsigned lane_id() { return threadIdx.x & 31u; }

// Scan one row for a neighbour satisfying `stop(u)`; lanes with short rows
// scan alone, longer rows are scanned by the whole warp.  Returns per lane.
template <class Stop>
__device__ __forceinline__ bool row_any(const uint32_t *__restrict__ ci, bool active, int64_t rs,
                                        int64_t re, uint32_t thread_max, Stop stop) {
    const int64_t deg = re - rs;
    const bool small = active && deg <= (int64_t)thread_max;
    const bool mid = active && !small;
    bool found = false;
    if (small) {
        for (int64_t e = rs; e < re; ++e)
            if (stop(ci[e], lane_id())) {
                found = true;
                break;
            }
    }
    unsigned mm = __ballot_sync(kFull, mid);
    const unsigned lane = lane_id();
    while (mm) {
        const int src = __ffs(mm) - 1;
        mm &= mm - 1;
        const int64_t ws = __shfl_sync(kFull, rs, src);
        const int64_t we = __shfl_sync(kFull, re, src);
        bool f = false;
        for (int64_t e0 = ws; e0 < we; e0 += 32) {
            const int64_t e = e0 + lane;
            bool hit = (e < we) && stop(ci[e], (unsigned)src);
            if (__any_sync(kFull, hit)) {
                f = true;
                break;
            }
        }
        if ((int)lane == src) found = f;
    }
    return found;
}

__global__ void __launch_bounds__(kBlock) k_phase_a(const int64_t *__restrict__ ro,
                                                    const uint32_t *__restrict__ ci,
                                                    uint32_t *S, uint32_t *const *lists,
                                                    unsigned long long *ctr, uint32_t t,
                                                    uint32_t key, uint32_t thread_max) {
    const unsigned long long len = ctr[kLen];
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        ctr[kCandLeft] = 0;
        if (len > 0) ctr[kBusy] += 1;
    }
    const uint32_t *L = lists[ctr[kCur] & 1];
    const uint32_t in_t = 2u * t;
    const unsigned lane = lane_id();
    const unsigned long long stride = (unsigned long long)gridDim.x * blockDim.x;
    for (unsigned long long base = (unsigned long long)blockIdx.x * blockDim.x + (threadIdx.x & ~31u);
         base < len; base += stride) {
        const unsigned long long idx = base + lane;
        uint32_t v = 0;
        bool cand = false;
        int64_t rs = 0, re = 0;
        if (idx < len) {
            v = L[idx];
            cand = S[v] == kCand;
            if (cand) {
                rs = ro[v];
                re = ro[v + 1];
            }
        }
        // the weight of each lane's own vertex (shuffled to the warp on demand)
        const uint32_t pv_lane = weight_mix(v ^ key);
        // Alg.3 L6-8: v joins iff no candidate neighbour has a larger weight
        bool joins = false;
        {
            const int64_t deg = re - rs;
            const bool small = cand && deg <= (int64_t)thread_max;
            const bool mid = cand && !small;
            if (small) {
                joins = true;
                for (int64_t e = rs; e < re; ++e) {
                    uint32_t u = ci[e];
                    uint32_t su = S[u];
                    if ((su == kCand || su == in_t) && weight_mix(u ^ key) > pv_lane) {
                        joins = false;
                        break;
                    }
                }
            }
            unsigned mm = __ballot_sync(kFull, mid);
            while (mm) {
                const int src = __ffs(mm) - 1;
                mm &= mm - 1;
                const int64_t ws = __shfl_sync(kFull, rs, src);
                const int64_t we = __shfl_sync(kFull, re, src);
                const uint32_t pw = __shfl_sync(kFull, pv_lane, src);
                bool beat = false;
                for (int64_t e0 = ws; e0 < we; e0 += 32) {
                    const int64_t e = e0 + lane;
                    bool hit = false;
                    if (e < we) {
                        uint32_t u = ci[e];
                        uint32_t su = S[u];
                        hit = (su == kCand || su == in_t) && weight_mix(u ^ key) > pw;
                    }
                    if (__any_sync(kFull, hit)) {
                        beat = true;
                        break;
                    }
                }
                if ((int)lane == src) joins = !beat;
            }
        }
        if (joins) S[v] = in_t;  // Alg.3 L10, L12
    }
}

__global__ void __launch_bounds__(kBlock) k_phase_b(const int64_t *__restrict__ ro,
                                                    const uint32_t *__restrict__ ci,
                                                    uint32_t *S, uint32_t *const *lists,
                                                    unsigned long long *ctr, uint32_t t,
                                                    uint32_t thread_max) {
    const unsigned long long len = ctr[kLen];
    const uint32_t *L = lists[ctr[kCur] & 1];
    const uint32_t in_t = 2u * t;
    const unsigned lane = lane_id();
    const unsigned long long stride = (unsigned long long)gridDim.x * blockDim.x;
    for (unsigned long long base = (unsigned long long)blockIdx.x * blockDim.x + (threadIdx.x & ~31u);
         base < len; base += stride) {
        const unsigned long long idx = base + lane;
        uint32_t v = 0;
        bool cand = false;
        int64_t rs = 0, re = 0;
        if (idx < len) {
            v = L[idx];
            cand = S[v] == kCand;
            if (cand) {
                rs = ro[v];
                re = ro[v + 1];
            }
        }
        // Alg.3 L19-20: drop candidates adjacent to a member that joined in t
        bool out = row_any(ci, cand, rs, re, thread_max,
                           [&](uint32_t u, unsigned) { return S[u] == in_t; });
        if (cand && out) S[v] = in_t + 1u;
        unsigned still = __ballot_sync(kFull, cand && !out);
        if (lane == 0 && still) atomicAdd(&ctr[kCandLeft], (unsigned long long)__popc(still));
    }
}

// Alg.2 L17 once the candidate set is exhausted: colour the members with c,
// move everyone else to the next list as a fresh candidate (R10).
__global__ void __launch_bounds__(kBlock) k_commit(uint32_t *C, uint32_t *S, uint32_t *const *lists,
                                                   unsigned long long *ctr) {
    const unsigned long long len = ctr[kLen];
    if (len == 0 || ctr[kCandLeft] != 0) return;  // uniform across the grid
    const unsigned cur = (unsigned)(ctr[kCur] & 1);
    const uint32_t *L = lists[cur];
    uint32_t *Lnext = lists[cur ^ 1];
    const uint32_t c = (uint32_t)ctr[kColor];
    const unsigned lane = lane_id();
    const unsigned long long stride = (unsigned long long)gridDim.x * blockDim.x;
    for (unsigned long long base = (unsigned long long)blockIdx.x * blockDim.x + (threadIdx.x & ~31u);
         base < len; base += stride) {
        const unsigned long long idx = base + lane;
        bool keep = false;
        uint32_t v = 0;
        if (idx < len) {
            v = L[idx];
            uint32_t sv = S[v];
            if ((sv & 1u) == 0u && sv != kCand) {
                C[v] = c;
            } else {
                S[v] = kCand;
                keep = true;
            }
        }
        unsigned m = __ballot_sync(kFull, keep);
        unsigned long long pos = 0;
        if (m) {
            if (lane == (unsigned)(__ffs(m) - 1)) pos = atomicAdd(&ctr[kNextLen], (unsigned long long)__popc(m));
            pos = __shfl_sync(kFull, pos, __ffs(m) - 1);
            if (keep) Lnext[pos + __popc(m & ((1u << lane) - 1u))] = v;
        }
    }
    // last block to finish publishes the next list
    __threadfence();
    __syncthreads();
    if (threadIdx.x == 0) {
        unsigned long long ticket = atomicAdd(&ctr[kTicket], 1ull);
        if (ticket == gridDim.x - 1) {
            __threadfence();
            unsigned long long nl = atomicAdd(&ctr[kNextLen], 0ull);
            ctr[kLen] = nl;
            ctr[kNextLen] = 0;
            ctr[kCur] = cur ^ 1u;
            ctr[kColor] = c + 1u;
            ctr[kTicket] = 0;
            ctr[kCandLeft] = 1;  // stays "busy" until the next phase B recounts
        }
    }
}

__global__ void k_iota_fill(uint32_t *L, uint32_t *S, int64_t n) {
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
         i += (int64_t)gridDim.x * blockDim.x) {
        L[i] = (uint32_t)i;
        S[i] = kCand;
    }
}

}  // namespace

int fill_u32(uint32_t *p, uint32_t val, int64_t n, cudaStream_t st);

int run_luby(gc_graph *g, const RunParams &p, RunResult *r) {
    Scratch &s = g->s;
    const int64_t n = g->n;
    r->rounds = r->inner = r->launches = 0;
    if (n == 0) return GC_OK;
    int rc = fill_u32(s.C, GC_UNC, n, g->stream);  // Alg.2 L3
    if (rc) return rc;
    const int blocks =
        (int)std::max<int64_t>(1, std::min<int64_t>((n + kBlock - 1) / kBlock, (int64_t)g->sm_count * 8));
    k_iota_fill<<<blocks, kBlock, 0, g->stream>>>(s.F[0], s.S, n);
    r->launches += 2;
    GC_CUDA_TRY(cudaMemsetAsync(s.ctr, 0, 16 * sizeof(unsigned long long), g->stream));
    unsigned long long init_len = (unsigned long long)n;
    GC_CUDA_TRY(cudaMemcpyAsync(s.ctr + kLen, &init_len, sizeof(init_len), cudaMemcpyHostToDevice,
                                g->stream));
    // device copy of the two list pointers
    uint32_t **lists = reinterpret_cast<uint32_t **>(s.ctr + 32);
    uint32_t *hl[2] = {s.F[0], s.F[1]};
    GC_CUDA_TRY(cudaMemcpyAsync(lists, hl, sizeof(hl), cudaMemcpyHostToDevice, g->stream));
    const uint32_t key = p.keys.k[0];
    int64_t t = 0;
    int64_t batch = p.batch_rounds > 0 ? p.batch_rounds : 4;
    for (;;) {
        for (int64_t b = 0; b < batch; ++b, ++t) {
            k_phase_a<<<blocks, kBlock, 0, g->stream>>>(g->ro, g->ci, s.S, lists, s.ctr,
                                                         (uint32_t)t, key,
                                                         (uint32_t)p.thread_deg_max);
            k_phase_b<<<blocks, kBlock, 0, g->stream>>>(g->ro, g->ci, s.S, lists, s.ctr,
                                                         (uint32_t)t, (uint32_t)p.thread_deg_max);
            k_commit<<<blocks, kBlock, 0, g->stream>>>(s.C, s.S, lists, s.ctr);
            r->launches += 3;
        }
        GC_CUDA_TRY(cudaGetLastError());
        GC_CUDA_TRY(cudaMemcpyAsync(s.host_pinned, s.ctr, 16 * sizeof(unsigned long long),
                                    cudaMemcpyDeviceToHost, g->stream));
        GC_CUDA_TRY(cudaStreamSynchronize(g->stream));
        const unsigned long long *h = reinterpret_cast<const unsigned long long *>(s.host_pinned);
        if (h[kLen] == 0) {
            r->rounds = (int64_t)h[kColor];
            r->inner = (int64_t)h[kBusy] + r->rounds;
            break;
        }
        if (2 * t > 0xFFFFFFF0ll) {
            set_error("Luby colouring exceeded the iteration limit");
            return GC_ERR_TOO_LARGE;
        }
        if (p.batch_rounds <= 0) batch = std::min<int64_t>(batch * 2, 128);
    }
    return GC_OK;
}

}  // namespace gc
