// gc_sweep.cu -- SWEEP mode of the max-min / multi-hash IS colouring.
//
// One round k of Alg.1 with the Alg.5 ColorOp:
// every vertex v of the frontier F_k (= uncoloured vertices, compacted) scans
// its neighbours u, counting only those still uncoloured at the start of the
// round, and records per hash j whether a larger (hi) or smaller (lo) weight
// exists (Alg.5 L29-34).  The scan stops once every hash has both (the answer
// can no longer change).  v then takes 2(kH+j)+1 if it has no smaller
// neighbour under the first such j (min), else 2(kH+j) (max) -- Alg.5 L37-42
// with R4/R8/R9.  Vertices that stay uncoloured are appended to F_{k+1}.
//
// In-place commit without atomics: the status test is the single
// unsigned compare C[u] >= 2kH (C = GC_UNC for uncoloured).  Colours written
// during round k are >= 2kH, older ones are < 2kH, so a neighbour coloured
// concurrently in this round still counts as active -- exactly the snapshot
// semantics of Alg.5 L26 (R6), whatever the interleaving.
//
// Load balance (the paper's serial per-thread loop is its stated flaw,
// P:L450-457): rows with deg <= thread_deg_max are scanned by one
// lane; longer rows by the whole warp, 32 coalesced column indices per step
// with a warp OR-reduction of the flag masks; rows >= hub_deg_min go to a hub
// list scanned by a whole CTA in a second kernel of the same round.
//
// Host control: rounds are enqueued in batches without host synchronisation;
// each kernel reads its frontier size from device memory, and rounds after
// completion are no-ops (an empty frontier), so the host reads the per-round
// sizes only once per batch.
#include "gc_internal.cuh"

namespace gc {

namespace {

constexpr int kBlock = 256;
constexpr unsigned kFull = 0xFFFFFFFFu;

// Counter slots in g->s.ctr (unsigned long long):
//   [0..2] frontier sizes, rotating with k % 3 (round k reads slot k%3,
//          appends to (k+1)%3 and clears (k+2)%3 for round k+1)
//   [3..5] hub-list sizes, rotating likewise
__device__ __forceinline__ unsigned lane_id() { return threadIdx.x & 31u; }

template <int HT>
struct Hashes {
    int H;
    __device__ __forceinline__ int count() const { return HT > 0 ? HT : H; }
};

// Per-neighbour update of the hi/lo bit masks over the hashes.
template <int HT>
__device__ __forceinline__ void visit(uint32_t u, const uint32_t *pv, const Keys &keys, int H,
                                      uint32_t &hi, uint32_t &lo) {
    const int nh = HT > 0 ? HT : H;
#pragma unroll
    for (int j = 0; j < (HT > 0 ? HT : GC_MAX_HASHES); ++j) {
        if (HT == 0 && j >= nh) break;
        uint32_t pu = weight_mix(u ^ keys.k[j]);
        hi |= (uint32_t)(pu > pv[j]) << j;
        lo |= (uint32_t)(pu < pv[j]) << j;
    }
}

template <int HT>
__device__ __forceinline__ void own_weights(uint32_t v, const Keys &keys, int H, uint32_t *pv) {
#pragma unroll
    for (int j = 0; j < (HT > 0 ? HT : GC_MAX_HASHES); ++j) {
        if (HT == 0 && j >= H) break;
        pv[j] = weight_mix(v ^ keys.k[j]);
    }
}

// Colour from the flag masks; returns GC_UNC if v stays blocked.
__device__ __forceinline__ uint32_t decide(uint32_t hi, uint32_t lo, uint32_t full, uint32_t k,
                                           int H) {
    uint32_t blocked = hi & lo;
    if (blocked == full) return GC_UNC;
    int j = __ffs(~blocked) - 1;  // smallest hash at which v is a max or a min
    uint32_t is_min = ((lo >> j) & 1u) ^ 1u;  // no smaller active neighbour
    return 2u * (k * (uint32_t)H + (uint32_t)j) + is_min;
}

// Warp-aggregated append of `v` (where pred) to list/counter.
__device__ __forceinline__ void warp_append(bool pred, uint32_t v, uint32_t *list,
                                            unsigned long long *counter) {
    unsigned m = __ballot_sync(kFull, pred);
    if (!m) return;
    unsigned lane = lane_id();
    unsigned leader = __ffs(m) - 1;
    unsigned long long base = 0;
    if (lane == leader) base = atomicAdd(counter, (unsigned long long)__popc(m));
    base = __shfl_sync(kFull, base, leader);
    if (pred) list[base + __popc(m & ((1u << lane) - 1u))] = v;
}

template <int HT, bool PROF>
__global__ void __launch_bounds__(kBlock) k_sweep(SweepArgs a) {
    const int64_t *__restrict__ ro = a.ro;
    const uint32_t *__restrict__ ci = a.ci;
    uint32_t *C = a.C;
    const uint32_t *__restrict__ Fin = a.Fin;
    uint32_t *__restrict__ Fout = a.Fout;
    uint32_t *__restrict__ hub = a.hub;
    unsigned long long *ctr = a.ctr;
    const uint32_t k = a.k, thread_max = a.thread_max, hub_min = a.hub_min, v0 = a.v0;
    const int H = a.H, dense = a.dense;
    const Keys &keys = a.keys;
    const int64_t n = a.n_loc;
    const unsigned long long N = dense ? (unsigned long long)n : ctr[k % 3];
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        ctr[(k + 2) % 3] = 0;
        ctr[3 + (k + 1) % 3] = 0;
        if ((int64_t)k < a.nk_cap) a.nk[k] = (int64_t)N;
    }
    const int nh = HT > 0 ? HT : H;
    const uint32_t full = (nh >= 32) ? kFull : ((1u << nh) - 1u);
    const uint32_t thresh = 2u * k * (uint32_t)nh;  // active iff C[u] >= thresh
    const unsigned lane = lane_id();
    const unsigned long long stride = (unsigned long long)gridDim.x * blockDim.x;
    for (unsigned long long base = (unsigned long long)blockIdx.x * blockDim.x + (threadIdx.x & ~31u);
         base < N; base += stride) {
        const unsigned long long idx = base + lane;
        const bool valid = idx < N;
        uint32_t v = 0;
        int64_t rs = 0, re = 0;
        if (valid) {
            v = dense ? v0 + (uint32_t)idx : Fin[idx];
            rs = ro[v - v0];
            re = ro[v - v0 + 1];
        }
        const int64_t deg = re - rs;
        const bool small = valid && deg <= (int64_t)thread_max;
        const bool big = valid && !small && deg >= (int64_t)hub_min;
        const bool mid = valid && !small && !big;
        uint32_t pv[HT > 0 ? HT : GC_MAX_HASHES];
        own_weights<HT>(v, keys, nh, pv);
        uint32_t hi = 0, lo = 0;
        uint32_t nvis = 0;  // PROF: neighbour entries examined by this lane
        if (small) {
            for (int64_t e = rs; e < re; ++e) {
                if (PROF) ++nvis;
                uint32_t u = ci[e];
                if (C[u] < thresh) continue;  // coloured before round k (Alg.5 L26)
                visit<HT>(u, pv, keys, nh, hi, lo);
                if ((hi & lo) == full) break;  // outcome fixed: blocked
            }
        }
        // rows of intermediate length: the whole warp scans one row at a time
        unsigned mm = __ballot_sync(kFull, mid);
        while (mm) {
            const int src = __ffs(mm) - 1;
            mm &= mm - 1;
            const uint32_t w = __shfl_sync(kFull, v, src);
            const int64_t ws = __shfl_sync(kFull, rs, src);
            const int64_t we = __shfl_sync(kFull, re, src);
            uint32_t pw[HT > 0 ? HT : GC_MAX_HASHES];
            own_weights<HT>(w, keys, nh, pw);
            uint32_t h = 0, l = 0;
            for (int64_t e0 = ws; e0 < we; e0 += 64) {
                const int64_t e1 = e0 + lane, e2 = e0 + 32 + lane;
                uint32_t u1 = e1 < we ? ci[e1] : 0u;
                uint32_t u2 = e2 < we ? ci[e2] : 0u;
                uint32_t c1 = e1 < we ? C[u1] : 0u;
                uint32_t c2 = e2 < we ? C[u2] : 0u;
                if (e1 < we && c1 >= thresh) visit<HT>(u1, pw, keys, nh, h, l);
                if (e2 < we && c2 >= thresh) visit<HT>(u2, pw, keys, nh, h, l);
                if (PROF) nvis += (e1 < we) + (e2 < we);
                h = __reduce_or_sync(kFull, h);
                l = __reduce_or_sync(kFull, l);
                if ((h & l) == full) break;
            }
            if ((int)lane == src) {
                hi = h;
                lo = l;
            }
        }
        // hubs: a CTA per row in k_hub
        warp_append(big, v, hub, &ctr[3 + k % 3]);
        const bool handled = small || mid;
        uint32_t col = GC_UNC;
        if (handled) {
            col = decide(hi, lo, full, k, nh);
            if (col != GC_UNC) C[v] = col;  // atomic-free commit (single writer)
        }
        warp_append(handled && col == GC_UNC, v, Fout, &ctr[(k + 1) % 3]);
        if (a.colored) {  // distributed: publish (v, colour) of this round
            const bool c = handled && col != GC_UNC;
            const unsigned m = __ballot_sync(kFull, c);
            if (m) {
                const unsigned leader = __ffs(m) - 1;
                unsigned long long b = 0;
                if (lane == leader) b = atomicAdd(&ctr[kColoredCtr], (unsigned long long)__popc(m));
                b = __shfl_sync(kFull, b, leader);
                if (c) a.colored[b + __popc(m & ((1u << lane) - 1u))] = make_uint2(v, col);
            }
        }
        if (PROF) {
            unsigned tot = __reduce_add_sync(kFull, nvis);
            if (lane == 0 && tot) atomicAdd(&ctr[20], (unsigned long long)tot);
        }
    }
}

// CTA-per-hub scan of round k.  Persistent over the hub list.
template <int HT, bool PROF>
__global__ void __launch_bounds__(512) k_hub(SweepArgs a) {
    const int64_t *__restrict__ ro = a.ro;
    const uint32_t *__restrict__ ci = a.ci;
    uint32_t *C = a.C;
    const uint32_t *__restrict__ hub = a.hub;
    uint32_t *__restrict__ Fout = a.Fout;
    unsigned long long *ctr = a.ctr;
    const uint32_t k = a.k, v0 = a.v0;
    const int H = a.H;
    const Keys &keys = a.keys;
    const unsigned long long nhub = ctr[3 + k % 3];
    const int nh = HT > 0 ? HT : H;
    const uint32_t full = (nh >= 32) ? kFull : ((1u << nh) - 1u);
    const uint32_t thresh = 2u * k * (uint32_t)nh;
    __shared__ uint32_t sh_hi, sh_lo;
    for (unsigned long long i = blockIdx.x; i < nhub; i += gridDim.x) {
        const uint32_t v = hub[i];
        const int64_t rs = ro[v - v0], re = ro[v - v0 + 1];
        uint32_t pv[HT > 0 ? HT : GC_MAX_HASHES];
        own_weights<HT>(v, keys, nh, pv);
        if (threadIdx.x == 0) {
            sh_hi = 0;
            sh_lo = 0;
        }
        __syncthreads();
        uint32_t h = 0, l = 0, H_all = 0, L_all = 0;
        uint32_t nvis = 0;
        constexpr int kUnroll = 4;
        for (int64_t e0 = rs; e0 < re; e0 += (int64_t)blockDim.x * kUnroll) {
            uint32_t u[kUnroll], c[kUnroll];
#pragma unroll
            for (int q = 0; q < kUnroll; ++q) {
                int64_t e = e0 + threadIdx.x + (int64_t)q * blockDim.x;
                u[q] = e < re ? ci[e] : 0u;
            }
#pragma unroll
            for (int q = 0; q < kUnroll; ++q) {
                int64_t e = e0 + threadIdx.x + (int64_t)q * blockDim.x;
                c[q] = e < re ? C[u[q]] : 0u;
            }
#pragma unroll
            for (int q = 0; q < kUnroll; ++q) {
                const bool in_row = (e0 + threadIdx.x + (int64_t)q * blockDim.x) < re;
                if (PROF) nvis += in_row;
                if (in_row && c[q] >= thresh) visit<HT>(u[q], pv, keys, nh, h, l);
            }
            h = __reduce_or_sync(kFull, h);
            l = __reduce_or_sync(kFull, l);
            if ((threadIdx.x & 31) == 0) {
                atomicOr(&sh_hi, h);
                atomicOr(&sh_lo, l);
            }
            __syncthreads();
            H_all = sh_hi;
            L_all = sh_lo;
            __syncthreads();
            if ((H_all & L_all) == full) break;
        }
        if (PROF) {
            unsigned tot = __reduce_add_sync(kFull, nvis);
            if ((threadIdx.x & 31) == 0 && tot) atomicAdd(&ctr[21], (unsigned long long)tot);
        }
        if (threadIdx.x == 0) {
            uint32_t col = decide(H_all, L_all, full, k, nh);
            if (col != GC_UNC) {
                C[v] = col;
                if (a.colored) a.colored[atomicAdd(&ctr[kColoredCtr], 1ull)] = make_uint2(v, col);
            } else {
                unsigned long long pos = atomicAdd(&ctr[(k + 1) % 3], 1ull);
                Fout[pos] = v;
            }
        }
        __syncthreads();
    }
}

__global__ void k_fill_u32(uint32_t *p, uint32_t val, int64_t n) {
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
         i += (int64_t)gridDim.x * blockDim.x)
        p[i] = val;
}

template <int HT, bool PROF>
int launch_round_args(const SweepArgs &a, cudaStream_t st, int blocks_sweep, int blocks_hub,
                      EventTimer *tm) {
    int rc = 0;
    if (PROF && (rc = tm->begin(st, 0))) return rc;
    k_sweep<HT, PROF><<<blocks_sweep, kBlock, 0, st>>>(a);
    if (PROF && (rc = tm->end(st))) return rc;
    if (PROF && (rc = tm->begin(st, 1))) return rc;
    k_hub<HT, PROF><<<blocks_hub, 512, 0, st>>>(a);
    if (PROF && (rc = tm->end(st))) return rc;
    return GC_OK;
}

template <int HT, bool PROF>
int launch_round(gc_graph *g, const RunParams &p, uint32_t k, int blocks_sweep, int blocks_hub,
                 EventTimer *tm) {
    Scratch &s = g->s;
    SweepArgs a;
    a.ro = g->ro;
    a.ci = g->ci;
    a.C = s.C;
    a.Fin = s.F[k & 1];
    a.Fout = s.F[(k + 1) & 1];
    a.hub = s.hub;
    a.ctr = s.ctr;
    a.nk = s.nk;
    a.nk_cap = s.nk_cap;
    a.k = k;
    a.H = p.H;
    a.keys = p.keys;
    a.dense = k == 0 ? 1 : 0;
    a.n_loc = g->n;
    a.v0 = 0;
    a.thread_max = (uint32_t)p.thread_deg_max;
    a.hub_min = (uint32_t)p.hub_deg_min;
    a.colored = nullptr;
    return launch_round_args<HT, PROF>(a, g->stream, blocks_sweep, blocks_hub, tm);
}

}  // namespace

EventTimer::~EventTimer() {
    for (auto e : ev) cudaEventDestroy(e);
}

int EventTimer::begin(cudaStream_t st, int klass) {
    if (used + 2 > ev.size()) {
        for (int i = 0; i < 2; ++i) {
            cudaEvent_t e;
            GC_CUDA_TRY(cudaEventCreate(&e));
            ev.push_back(e);
        }
        cls.push_back(0);
    }
    cls[used / 2] = klass;
    GC_CUDA_TRY(cudaEventRecord(ev[used], st));
    used++;
    return GC_OK;
}

int EventTimer::end(cudaStream_t st) {
    GC_CUDA_TRY(cudaEventRecord(ev[used], st));
    used++;
    return GC_OK;
}

int EventTimer::drain(Profile *p) {
    for (size_t i = 0; i + 1 < used; i += 2) {
        float ms = 0.f;
        GC_CUDA_TRY(cudaEventElapsedTime(&ms, ev[i], ev[i + 1]));
        p->ms[cls[i / 2]] += ms;
        p->launches[cls[i / 2]] += 1;
        p->launch_us.push_back(1e3f * ms);
    }
    used = 0;
    return GC_OK;
}

int sweep_round(const SweepArgs &a, cudaStream_t st, int blocks_sweep, int blocks_hub) {
    EventTimer tm;
    int rc = a.H == 1 ? launch_round_args<1, false>(a, st, blocks_sweep, blocks_hub, &tm)
                      : launch_round_args<0, false>(a, st, blocks_sweep, blocks_hub, &tm);
    if (rc) return rc;
    GC_CUDA_TRY(cudaGetLastError());
    return GC_OK;
}

int fill_u32(uint32_t *p, uint32_t val, int64_t n, cudaStream_t st) {
    if (n <= 0) return GC_OK;
    int blocks = (int)std::min<int64_t>((n + 255) / 256, 148 * 16);
    k_fill_u32<<<blocks, 256, 0, st>>>(p, val, n);
    GC_CUDA_TRY(cudaGetLastError());
    return GC_OK;
}

// Grow the per-round statistics array on the host side of a batch boundary.
int ensure_nk(gc_graph *g, int64_t need);

int run_sweep_maxmin(gc_graph *g, const RunParams &p, RunResult *r) {
    Scratch &s = g->s;
    const int64_t n = g->n;
    r->rounds = 0;
    r->launches = 0;
    if (n == 0) return GC_OK;
    int rc = fill_u32(s.C, GC_UNC, n, g->stream);  // Alg.5 L5
    if (rc) return rc;
    r->launches++;
    GC_CUDA_TRY(cudaMemsetAsync(s.ctr, 0, 24 * sizeof(unsigned long long), g->stream));
    // grid: enough warps for the first (dense) round, capped at 8 CTAs/SM resident
    const int blocks_sweep = (int)std::max<int64_t>(
        1, std::min<int64_t>((n + kBlock - 1) / kBlock, (int64_t)g->sm_count * 8));
    const int blocks_hub = g->sm_count * 2;
    int64_t k = 0;
    int64_t batch = p.batch_rounds > 0 ? p.batch_rounds : 4;
    const bool prof = p.prof && p.prof->on;
    EventTimer tm;
    for (;;) {
        rc = ensure_nk(g, k + batch + 1);
        if (rc) return rc;
        for (int64_t b = 0; b < batch; ++b, ++k) {
            if (p.H == 1)
                rc = prof ? launch_round<1, true>(g, p, (uint32_t)k, blocks_sweep, blocks_hub, &tm)
                          : launch_round<1, false>(g, p, (uint32_t)k, blocks_sweep, blocks_hub, &tm);
            else
                rc = prof ? launch_round<0, true>(g, p, (uint32_t)k, blocks_sweep, blocks_hub, &tm)
                          : launch_round<0, false>(g, p, (uint32_t)k, blocks_sweep, blocks_hub, &tm);
            if (rc) return rc;
            r->launches += 2;
        }
        GC_CUDA_TRY(cudaGetLastError());
        // read N_{k-batch} .. N_{k-1}; the first zero marks completion
        GC_CUDA_TRY(cudaMemcpyAsync(s.host_pinned, s.nk + (k - batch), sizeof(int64_t) * batch,
                                    cudaMemcpyDeviceToHost, g->stream));
        GC_CUDA_TRY(cudaStreamSynchronize(g->stream));
        if (prof && (rc = tm.drain(p.prof))) return rc;
        int64_t done_at = -1;
        for (int64_t b = 0; b < batch; ++b)
            if (s.host_pinned[b] == 0) {
                done_at = k - batch + b;
                break;
            }
        if (done_at >= 0) {
            r->rounds = done_at;
            break;
        }
        if (p.max_rounds > 0 && k >= p.max_rounds) {
            set_error("max-min colouring exceeded the round limit");
            return GC_ERR_TOO_LARGE;
        }
        if (p.batch_rounds <= 0) batch = std::min<int64_t>(batch * 2, 256);
    }
    r->inner = r->rounds;
    if (prof) {
        // algorithmic bytes: per round k the sweep reads the
        // frontier (4 N_k, not in the dense round 0) and the row offsets
        // (16 N_k), writes colours (4 Q_k) and the next frontier (4 N_{k+1});
        // every visited entry reads 4 B of col_indices.
        std::vector<int64_t> nk(r->rounds + 1, 0);
        if (r->rounds > 0)
            GC_CUDA_TRY(cudaMemcpy(nk.data(), s.nk, sizeof(int64_t) * r->rounds,
                                   cudaMemcpyDeviceToHost));
        unsigned long long vis[2] = {0, 0};
        GC_CUDA_TRY(cudaMemcpy(vis, s.ctr + 20, sizeof(vis), cudaMemcpyDeviceToHost));
        int64_t b = 0;
        for (int64_t kk = 0; kk < r->rounds; ++kk) {
            int64_t q = nk[kk] - nk[kk + 1];
            b += (kk > 0 ? 4 : 0) * nk[kk] + 16 * nk[kk] + 4 * q + 4 * nk[kk + 1];
        }
        p.prof->bytes[0] += b + 4 * (int64_t)vis[0];
        p.prof->bytes[1] += 4 * (int64_t)vis[1];
        p.prof->visits += (int64_t)(vis[0] + vis[1]);
    }
    return GC_OK;
}

}  // namespace gc
