// gc_api.cu -- the C ABI declared in include/gc.h: handle lifecycle, input
// validation, variant dispatch, output and colour counting.
#include <algorithm>
#include <cstdio>
#include <cstring>
#include <new>
#include <string>

#include "gc_internal.cuh"

namespace gc {

static thread_local std::string g_last_error;

void set_error(const std::string &msg) { g_last_error = msg; }

int cuda_fail(cudaError_t e, const char *what) {
    char buf[512];
    snprintf(buf, sizeof(buf), "CUDA error %s (%s) in %s", cudaGetErrorName(e),
             cudaGetErrorString(e), what);
    set_error(buf);
    cudaGetLastError();  // clear sticky-free errors
    return e == cudaErrorMemoryAllocation ? GC_ERR_OOM : GC_ERR_CUDA;
}

bool is_device_ptr(const void *p) {
    if (!p) return false;
    cudaPointerAttributes a;
    if (cudaPointerGetAttributes(&a, p) != cudaSuccess) {
        cudaGetLastError();
        return false;
    }
    return a.type == cudaMemoryTypeDevice || a.type == cudaMemoryTypeManaged;
}

namespace {

constexpr int kCtrWords = 64;

__global__ void k_validate(const int64_t *__restrict__ ro, const uint32_t *__restrict__ ci,
                           int64_t n, int64_t nnz, int64_t n_global, int64_t v_begin,
                           unsigned long long *err) {
    // err[0]: non-monotone / out-of-range offsets; err[1]: col >= n; err[2]: self-loop;
    // err[3]: max degree.  Rows of <= 32 entries are checked by one lane, longer
    // rows by the whole warp (coalesced); counts are warp-aggregated.
    const unsigned lane = threadIdx.x & 31u;
    unsigned long long bad_off = 0, bad_col = 0, loops = 0, maxdeg = 0;
    const int64_t stride = (int64_t)gridDim.x * blockDim.x;
    for (int64_t base = (int64_t)blockIdx.x * blockDim.x + (threadIdx.x & ~31u); base < n;
         base += stride) {
        const int64_t v = base + lane;
        int64_t a0 = 0, b0 = 0;
        bool ok = false;
        if (v < n) {
            a0 = ro[v];
            b0 = ro[v + 1];
            ok = a0 <= b0 && a0 >= 0 && b0 <= nnz;
            if (!ok) ++bad_off;
            else maxdeg = max(maxdeg, (unsigned long long)(b0 - a0));
        }
        const bool shortrow = ok && b0 - a0 <= 32;
        if (shortrow)
            for (int64_t e = a0; e < b0; ++e) {
                const uint32_t u = ci[e];
                if ((int64_t)u >= n_global) ++bad_col;
                else if ((int64_t)u == v + v_begin) ++loops;
            }
        unsigned lm = __ballot_sync(0xFFFFFFFFu, ok && !shortrow);
        while (lm) {
            const int src = __ffs(lm) - 1;
            lm &= lm - 1;
            const int64_t ws = __shfl_sync(0xFFFFFFFFu, a0, src);
            const int64_t we = __shfl_sync(0xFFFFFFFFu, b0, src);
            const int64_t wv = __shfl_sync(0xFFFFFFFFu, v, src);
            for (int64_t e = ws + lane; e < we; e += 32) {
                const uint32_t u = ci[e];
                if ((int64_t)u >= n_global) ++bad_col;
                else if ((int64_t)u == wv + v_begin) ++loops;
            }
        }
    }
    bad_off = __reduce_add_sync(0xFFFFFFFFu, (unsigned)bad_off);
    bad_col = __reduce_add_sync(0xFFFFFFFFu, (unsigned)min(bad_col, 1ull << 20));
    loops = __reduce_add_sync(0xFFFFFFFFu, (unsigned)min(loops, 1ull << 20));
    const unsigned md_hi = __reduce_max_sync(0xFFFFFFFFu, (unsigned)(maxdeg >> 32));
    const unsigned md_lo = __reduce_max_sync(0xFFFFFFFFu, (unsigned)((maxdeg >> 32) == md_hi ? maxdeg : 0));
    if (lane == 0) {
        if (bad_off) atomicAdd(&err[0], bad_off);
        if (bad_col) atomicAdd(&err[1], bad_col);
        if (loops) atomicAdd(&err[2], loops);
        atomicMax(&err[3], ((unsigned long long)md_hi << 32) | md_lo);
    }
}

// Symmetry: for every entry (v,u) some entry (u,v) exists.  Linear scan of
// row u (rows may be unsorted); O(sum deg^2) worst case, opt-in only.
__global__ void k_validate_sym(const int64_t *__restrict__ ro, const uint32_t *__restrict__ ci,
                               int64_t n, unsigned long long *err) {
    const int lane = threadIdx.x & 31;
    const int64_t warp = ((int64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const int64_t nwarps = ((int64_t)gridDim.x * blockDim.x) >> 5;
    for (int64_t v = warp; v < n; v += nwarps) {
        for (int64_t e = ro[v]; e < ro[v + 1]; ++e) {
            uint32_t u = ci[e];
            bool found = false;
            for (int64_t f0 = ro[u]; f0 < ro[u + 1]; f0 += 32) {
                int64_t f = f0 + lane;
                bool hit = f < ro[u + 1] && ci[f] == (uint32_t)v;
                if (__any_sync(0xFFFFFFFFu, hit)) {
                    found = true;
                    break;
                }
            }
            if (!found && lane == 0) atomicAdd(&err[4], 1ull);
        }
    }
}

__global__ void k_priorities(uint64_t v_begin, int64_t count, uint32_t key, uint32_t *out) {
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < count;
         i += (int64_t)gridDim.x * blockDim.x)
        out[i] = weight_mix((uint32_t)(v_begin + (uint64_t)i) ^ key);
}

__global__ void k_max_u32(const uint32_t *__restrict__ C, int64_t n, unsigned long long *mx) {
    uint32_t m = 0;
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
         i += (int64_t)gridDim.x * blockDim.x)
        m = max(m, C[i]);
    m = __reduce_max_sync(0xFFFFFFFFu, m);
    if ((threadIdx.x & 31) == 0) atomicMax(mx, (unsigned long long)m);
}

__global__ void k_mark(const uint32_t *__restrict__ C, int64_t n, uint32_t *bitmap) {
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
         i += (int64_t)gridDim.x * blockDim.x) {
        uint32_t c = C[i];
        uint32_t bit = 1u << (c & 31);
        if (!(bitmap[c >> 5] & bit)) atomicOr(&bitmap[c >> 5], bit);
    }
}

// the same with the block's share of the used-colour set in shared memory
// (every SM otherwise keeps re-issuing atomics on the few hundred global
// words: its L1 copy of a word never shows other SMs' bits); one OR per
// non-zero word and block at the end
constexpr int64_t kMarkSmemWords = 12288;  // 48 KB: colours < 393,216
__global__ void k_mark_sm(const uint32_t *__restrict__ C, int64_t n, uint32_t *bitmap, int64_t words) {
    extern __shared__ uint32_t sb[];
    for (int64_t i = threadIdx.x; i < words; i += blockDim.x) sb[i] = 0u;
    __syncthreads();
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
         i += (int64_t)gridDim.x * blockDim.x) {
        const uint32_t c = C[i];
        const uint32_t bit = 1u << (c & 31);
        if (!(sb[c >> 5] & bit)) atomicOr(&sb[c >> 5], bit);
    }
    __syncthreads();
    for (int64_t i = threadIdx.x; i < words; i += blockDim.x)
        if (sb[i]) atomicOr(&bitmap[i], sb[i]);
}

__global__ void k_popc(const uint32_t *__restrict__ bitmap, int64_t words, unsigned long long *cnt) {
    unsigned long long s = 0;
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < words;
         i += (int64_t)gridDim.x * blockDim.x)
        s += __popc(bitmap[i]);
    s = __reduce_add_sync(0xFFFFFFFFu, (unsigned)s);
    if ((threadIdx.x & 31) == 0 && s) atomicAdd(cnt, s);
}

// Exclusive prefix of popcounts over the bitmap words (single CTA; the
// bitmap has <= 2^27 words so this loops in chunks), then rank lookup.
__global__ void k_rank_words(const uint32_t *__restrict__ bitmap, int64_t words, uint32_t *rank) {
    __shared__ uint32_t carry;
    __shared__ uint32_t warp_sums[32];
    if (threadIdx.x == 0) carry = 0;
    __syncthreads();
    for (int64_t base = 0; base < words; base += blockDim.x) {
        int64_t i = base + threadIdx.x;
        uint32_t x = i < words ? (uint32_t)__popc(bitmap[i]) : 0u;
        // inclusive warp scan
        uint32_t y = x;
        for (int d = 1; d < 32; d <<= 1) {
            uint32_t z = __shfl_up_sync(0xFFFFFFFFu, y, d);
            if ((threadIdx.x & 31) >= d) y += z;
        }
        if ((threadIdx.x & 31) == 31) warp_sums[threadIdx.x >> 5] = y;
        __syncthreads();
        if (threadIdx.x < 32) {
            uint32_t w = threadIdx.x < (blockDim.x >> 5) ? warp_sums[threadIdx.x] : 0u;
            uint32_t ws = w;
            for (int d = 1; d < 32; d <<= 1) {
                uint32_t z = __shfl_up_sync(0xFFFFFFFFu, ws, d);
                if (threadIdx.x >= d) ws += z;
            }
            warp_sums[threadIdx.x] = ws - w;  // exclusive
        }
        __syncthreads();
        uint32_t excl = carry + warp_sums[threadIdx.x >> 5] + (y - x);
        if (i < words) rank[i] = excl;
        __syncthreads();
        if (threadIdx.x == blockDim.x - 1) carry = excl + x;
        __syncthreads();
    }
}

__global__ void k_remap(uint32_t *C, int64_t n, const uint32_t *__restrict__ bitmap,
                        const uint32_t *__restrict__ rank) {
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
         i += (int64_t)gridDim.x * blockDim.x) {
        uint32_t c = C[i];
        uint32_t w = c >> 5, b = c & 31;
        C[i] = rank[w] + (uint32_t)__popc(bitmap[w] & ((1u << b) - 1u));
    }
}

int grid_for(int64_t n, int sm) {
    return (int)std::max<int64_t>(1, std::min<int64_t>((n + 255) / 256, (int64_t)sm * 8));
}

int current_device_ok(int *dev, int *sms) {
    int count = 0;
    cudaError_t e = cudaGetDeviceCount(&count);
    if (e != cudaSuccess || count == 0) {
        cudaGetLastError();
        set_error("no CUDA device available (libgc has no CPU fallback)");
        return GC_ERR_CUDA;
    }
    GC_CUDA_TRY(cudaGetDevice(dev));
    GC_CUDA_TRY(cudaDeviceGetAttribute(sms, cudaDevAttrMultiProcessorCount, *dev));
    int major = 0;
    GC_CUDA_TRY(cudaDeviceGetAttribute(&major, cudaDevAttrComputeCapabilityMajor, *dev));
    if (major < 10) {
        set_error("libgc is built for sm_100a (Blackwell B200); this device is older");
        return GC_ERR_CUDA;
    }
    return GC_OK;
}

}  // namespace

int fill_u32(uint32_t *p, uint32_t val, int64_t n, cudaStream_t st);

int ensure_nk(gc_graph *g, int64_t need) {
    Scratch &s = g->s;
    if (need <= s.nk_cap) return GC_OK;
    int64_t cap = std::max<int64_t>(need * 2, 1 << 12);
    int64_t *nk = nullptr, *rstat = nullptr;
    GC_CUDA_TRY(dmalloc(&nk, sizeof(int64_t) * cap));
    GC_CUDA_TRY(dmalloc(&rstat, sizeof(int64_t) * 16 * cap));
    GC_CUDA_TRY(cudaMemsetAsync(rstat, 0, sizeof(int64_t) * 16 * cap, g->stream));
    if (s.nk) {
        GC_CUDA_TRY(cudaMemcpyAsync(nk, s.nk, sizeof(int64_t) * s.nk_cap, cudaMemcpyDeviceToDevice,
                                    g->stream));
        GC_CUDA_TRY(cudaMemcpyAsync(rstat, s.rstat, sizeof(int64_t) * 16 * s.nk_cap,
                                    cudaMemcpyDeviceToDevice, g->stream));
        GC_CUDA_TRY(cudaStreamSynchronize(g->stream));
        dfree(s.nk);
        dfree(s.rstat);
    }
    s.nk = nk;
    s.rstat = rstat;
    s.nk_cap = cap;
    return GC_OK;
}

int ensure_scratch(gc_graph *g, bool need_event, bool need_luby) {
    Scratch &s = g->s;
    const size_t nn = (size_t)std::max<int64_t>(g->n, 1);
    if (!s.C) {
        GC_CUDA_TRY(dmalloc(&s.C, nn * 4));
        GC_CUDA_TRY(dmalloc(&s.F[0], nn * 4));
        GC_CUDA_TRY(dmalloc(&s.F[1], nn * 4));
        GC_CUDA_TRY(dmalloc(&s.hub, nn * 4));
        GC_CUDA_TRY(dmalloc(&s.ctr, kCtrWords * sizeof(unsigned long long)));
        GC_CUDA_TRY(cudaMemset(s.ctr, 0, kCtrWords * sizeof(unsigned long long)));
        GC_CUDA_TRY(hmalloc(&s.host_pinned, 4096));
        int rc = ensure_nk(g, 1 << 12);
        if (rc) return rc;
    }
    if ((need_luby || need_event) && !s.S) GC_CUDA_TRY(dmalloc(&s.S, nn * 4));
    if (need_event && !s.W) {
        GC_CUDA_TRY(dmalloc(&s.W, nn * 8));
        GC_CUDA_TRY(dmalloc(&s.P, nn * 8));
        GC_CUDA_TRY(dmalloc(&s.Q, nn * 4));
        // long-row notify items (u, segment): at most n + nnz/128 per round
        GC_CUDA_TRY(dmalloc(&s.Q2, (nn + (size_t)g->nnz / 128 + 1) * 8));
        GC_CUDA_TRY(dmalloc(&s.Q3, (nn + (size_t)g->nnz / 128 + 1) * 8));
        GC_CUDA_TRY(dmalloc(&s.LS, nn * 32));
        GC_CUDA_TRY(dmalloc(&s.M, ((nn + 31) / 32) * 4));
    }
    return GC_OK;
}

// Distinct colours of C[0..n); optionally renumber in place (R12).
int64_t count_colors_device(gc_graph *g, const uint32_t *C, int64_t n, bool compact,
                            uint32_t *C_inout, int64_t *launches, int64_t max_hint) {
    if (n == 0) return 0;
    Scratch &s = g->s;
    cudaStream_t st = g->stream;
    unsigned long long *tmp = s.ctr + 48;
    GC_CUDA_TRY(cudaMemsetAsync(tmp, 0, 2 * sizeof(unsigned long long), st));
    const int grid = grid_for(n, g->sm_count);
    uint64_t maxc;
    if (max_hint >= 0) {  // (the colouring kernel computed it: no pass, no host round trip)
        maxc = (uint64_t)max_hint;
    } else {
        k_max_u32<<<grid, 256, 0, st>>>(C, n, tmp);
        GC_CUDA_TRY(cudaMemcpyAsync(s.host_pinned, tmp, sizeof(unsigned long long),
                                    cudaMemcpyDeviceToHost, st));
        GC_CUDA_TRY(cudaStreamSynchronize(st));
        maxc = *reinterpret_cast<unsigned long long *>(s.host_pinned);
    }
    if (maxc == GC_UNC) {
        set_error("internal: uncoloured vertex in the result");
        return GC_ERR_CUDA;
    }
    const int64_t words = (int64_t)(maxc >> 5) + 1;
    if (words > s.bitmap_words) {
        if (s.bitmap) dfree(s.bitmap);
        s.bitmap = nullptr;
        GC_CUDA_TRY(dmalloc(&s.bitmap, (size_t)words * 8));  // bitmap + rank table
        s.bitmap_words = words;
    }
    uint32_t *rank = s.bitmap + words;
    GC_CUDA_TRY(cudaMemsetAsync(s.bitmap, 0, (size_t)words * 4, st));
    if (words <= kMarkSmemWords) {
        if (words * 4 > 48 * 1024)
            GC_CUDA_TRY(cudaFuncSetAttribute(k_mark_sm, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)(words * 4)));
        k_mark_sm<<<std::min<int>(grid, g->sm_count * 4), 512, (size_t)words * 4, st>>>(C, n, s.bitmap, words);
    } else {
        k_mark<<<grid, 256, 0, st>>>(C, n, s.bitmap);
    }
    k_popc<<<grid_for(words, g->sm_count), 256, 0, st>>>(s.bitmap, words, tmp + 1);
    *launches += 3;
    if (compact) {
        k_rank_words<<<1, 1024, 0, st>>>(s.bitmap, words, rank);
        k_remap<<<grid, 256, 0, st>>>(C_inout, n, s.bitmap, rank);
        *launches += 2;
    }
    GC_CUDA_TRY(cudaGetLastError());
    GC_CUDA_TRY(cudaMemcpyAsync(s.host_pinned, tmp + 1, sizeof(unsigned long long),
                                cudaMemcpyDeviceToHost, st));
    GC_CUDA_TRY(cudaStreamSynchronize(st));
    return (int64_t)*reinterpret_cast<unsigned long long *>(s.host_pinned);
}

int launch_priorities(uint64_t seed, int j, int64_t v_begin, int64_t count, uint32_t *out,
                      cudaStream_t st) {
    if (count <= 0) return GC_OK;
    k_priorities<<<grid_for(count, 148), 256, 0, st>>>((uint64_t)v_begin, count,
                                                      weight_key(seed, j), out);
    GC_CUDA_TRY(cudaGetLastError());
    return GC_OK;
}

static void free_scratch(Scratch &s) {
    dfree(s.C);
    dfree(s.F[0]);
    dfree(s.F[1]);
    dfree(s.hub);
    dfree(s.S);
    dfree(s.W);
    dfree(s.P);
    dfree(s.Q);
    dfree(s.Q2);
    dfree(s.Q3);
    dfree(s.LS);
    dfree(s.M);
    dfree(s.ctr);
    dfree(s.nk);
    dfree(s.rstat);
    dfree(s.bitmap);
    dfree(s.hist);
    dfree(s.cnt);
    dfree(s.cnt32);
    dfree(s.big);
    dfree(s.big32);
    dfree(s.Z);
    dfree(s.SL);
    dfree(s.WL);
    dfree(s.hubs);
    dfree(s.cctr);
    dfree(s.jslot);
    dfree(s.deg);
    dfree(s.jcr);
    dfree(s.cM);
    dfree(s.crow);
    if (s.host_pinned) hfree(s.host_pinned);
    s = Scratch();
}

void destroy_dist(gc_graph *g);  // gc_dist.cu

}  // namespace gc

using namespace gc;

extern "C" {

const char *gc_last_error(void) { return g_last_error.c_str(); }

const char *gc_version(void) {
    static char buf[64];
    if (!buf[0]) snprintf(buf, sizeof(buf), "gc %d sm_100a cudart %d", GC_ABI_VERSION, CUDART_VERSION);
    return buf;
}

int gc_create_csr_internal(int64_t n, int64_t nnz, const int64_t *row_offsets,
                           const uint32_t *col_indices, uint32_t flags, gc_graph **out,
                           int64_t v_begin, int64_t n_global) {
    if (!out) {
        set_error("gc_create_csr: out is NULL");
        return GC_ERR_INVALID_ARG;
    }
    *out = nullptr;
    if (n < 0 || nnz < 0 || !row_offsets || (nnz > 0 && !col_indices)) {
        set_error("gc_create_csr: bad sizes or NULL arrays");
        return GC_ERR_INVALID_ARG;
    }
    if (n_global >= (int64_t)1 << 32) {
        set_error("gc_create_csr: n must be < 2^32 (uint32 vertex ids)");
        return GC_ERR_TOO_LARGE;
    }
    int dev = 0, sms = 148;
    int rc = current_device_ok(&dev, &sms);
    if (rc) return rc;
    gc_graph *g = new (std::nothrow) gc_graph();
    if (!g) return GC_ERR_OOM;
    g->device = dev;
    g->sm_count = sms;
    g->n = n;
    g->n_global = n_global;
    g->v_begin = v_begin;
    g->nnz = nnz;
    const bool ro_dev = is_device_ptr(row_offsets);
    const bool ci_dev = nnz == 0 || is_device_ptr(col_indices);
    auto fail = [&](int code) {
        if (g->owns_csr) {
            dfree(g->ro);
            dfree(g->ci);
        }
        free_scratch(g->s);
        delete g;
        return code;
    };
    if ((flags & GC_BORROW_DEVICE) && ro_dev && ci_dev) {
        g->owns_csr = false;
        g->ro = const_cast<int64_t *>(row_offsets);
        g->ci = const_cast<uint32_t *>(col_indices);
    } else {
        cudaError_t e = dmalloc(&g->ro, sizeof(int64_t) * (size_t)(n + 1));
        if (e == cudaSuccess) e = dmalloc(&g->ci, sizeof(uint32_t) * (size_t)std::max<int64_t>(nnz, 1));
        if (e != cudaSuccess) return fail(cuda_fail(e, "dmalloc(csr)"));
        e = cudaMemcpy(g->ro, row_offsets, sizeof(int64_t) * (size_t)(n + 1), cudaMemcpyDefault);
        if (e == cudaSuccess && nnz > 0)
            e = cudaMemcpy(g->ci, col_indices, sizeof(uint32_t) * (size_t)nnz, cudaMemcpyDefault);
        if (e != cudaSuccess) return fail(cuda_fail(e, "cudaMemcpy(csr)"));
    }
    // validation on the device
    rc = ensure_scratch(g, false, false);
    if (rc) return fail(rc);
    int64_t first = 0, last = 0;
    cudaError_t e = cudaMemcpy(&first, g->ro, sizeof(int64_t), cudaMemcpyDeviceToHost);
    if (e == cudaSuccess)
        e = cudaMemcpy(&last, g->ro + n, sizeof(int64_t), cudaMemcpyDeviceToHost);
    if (e != cudaSuccess) return fail(cuda_fail(e, "cudaMemcpy(offsets)"));
    if (first != 0 || last != nnz) {
        set_error("gc_create_csr: row_offsets[0] must be 0 and row_offsets[n] == nnz");
        return fail(GC_ERR_INVALID_ARG);
    }
    unsigned long long *err = g->s.ctr + 40;
    e = cudaMemset(err, 0, 8 * sizeof(unsigned long long));
    if (e != cudaSuccess) return fail(cuda_fail(e, "cudaMemset"));
    if (n > 0) {
        // the distributed path checks col < n_global (ghost ids are global)
        k_validate<<<grid_for(n, sms), 256>>>(g->ro, g->ci, n, nnz, n_global, v_begin, err);
        if ((flags & GC_VALIDATE) && n == n_global)
            k_validate_sym<<<grid_for(n * 32, sms), 256>>>(g->ro, g->ci, n, err);
    }
    unsigned long long herr[8] = {0};
    e = cudaMemcpy(herr, err, sizeof(herr), cudaMemcpyDeviceToHost);
    if (e != cudaSuccess) return fail(cuda_fail(e, "validate"));
    if (herr[0]) {
        set_error("gc_create_csr: row_offsets are not monotone / in range");
        return fail(GC_ERR_INVALID_ARG);
    }
    if (herr[1]) {
        set_error("gc_create_csr: column index >= n");
        return fail(GC_ERR_INVALID_ARG);
    }
    if (herr[2]) {
        set_error("gc_create_csr: self-loop (never terminates; R7)");
        return fail(GC_ERR_SELF_LOOP);
    }
    if (herr[4]) {
        set_error("gc_create_csr: adjacency is not symmetric");
        return fail(GC_ERR_NOT_SYMMETRIC);
    }
    g->max_deg = (int64_t)herr[3];
    *out = g;
    return GC_OK;
}

int gc_create_csr(int64_t n, int64_t nnz, const int64_t *row_offsets, const uint32_t *col_indices,
                  uint32_t flags, gc_graph **out) {
    NvtxRange nv_("gc_create_csr");
    return gc_create_csr_internal(n, nnz, row_offsets, col_indices, flags, out, 0, n);
}

int gc_set_stream(gc_graph *g, void *cuda_stream) {
    if (!g) {
        set_error("gc_set_stream: NULL handle");
        return GC_ERR_INVALID_ARG;
    }
    g->stream = (cudaStream_t)cuda_stream;
    return GC_OK;
}

void gc_destroy(gc_graph *g) {
    if (!g) return;
    cudaSetDevice(g->device);
    // blocks go back to the library cache (gc_alloc.cu), so no work that
    // uses them may still be pending (cudaFree used to imply this sync)
    cudaDeviceSynchronize();
    destroy_dist(g);
    if (g->owns_csr) {
        dfree(g->ro);
        dfree(g->ci);
    }
    free_scratch(g->s);
    delete g;
}

int64_t gc_color_dist(gc_graph *g, const gc_options *o, int32_t *colors_out, gc_stats *stats);

int64_t gc_color_ex(gc_graph *g, const gc_options *o, int32_t *colors_out, gc_stats *stats) {
    NvtxRange nv_("gc_color");
    if (!g || !o || o->struct_size < sizeof(gc_options)) {
        set_error("gc_color_ex: NULL handle/options or options.struct_size too small");
        return GC_ERR_INVALID_ARG;
    }
    if (g->n > 0 && !colors_out) {
        set_error("gc_color_ex: colors_out is NULL");
        return GC_ERR_INVALID_ARG;
    }
    if (stats && stats->struct_size < sizeof(gc_stats)) {
        set_error("gc_color_ex: stats.struct_size too small");
        return GC_ERR_INVALID_ARG;
    }
    const int kind = GC_VARIANT_KIND(o->variant);
    int H = 1;
    if (kind == GC_MULTIHASH(0)) {
        H = GC_VARIANT_HASHES(o->variant);
        if (H < 1 || H > GC_MAX_HASHES) {
            set_error("gc_color_ex: multi-hash needs 1 <= h <= 16");
            return GC_ERR_INVALID_ARG;
        }
    } else if (kind == GC_HASH_IS(0)) {
        if (GC_VARIANT_HASHES(o->variant) > GC_HASH_TABLE_MAX) {
            set_error("gc_color_ex: hash IS needs a table of 0..64 colours");
            return GC_ERR_INVALID_ARG;
        }
    } else if (kind != GC_MAXMIN && kind != GC_LUBY_MIS && kind != GC_IS_ALG2 && kind != GC_JP_ALG4) {
        set_error("gc_color_ex: unknown variant");
        return GC_ERR_INVALID_ARG;
    }
    if (o->mode < GC_MODE_AUTO || o->mode > GC_MODE_COUNT) {
        set_error("gc_color_ex: unknown mode");
        return GC_ERR_INVALID_ARG;
    }
    const int ldf = GC_VARIANT_LDF(o->variant) ? 1 : 0;
    if ((o->variant & ~(0xFFFF | GC_LDF(0))) != 0 ||
        (ldf && (kind == GC_MULTIHASH(0) || kind == GC_HASH_IS(0)))) {
        set_error("gc_color_ex: bad variant flags (GC_LDF applies to GC_MAXMIN, GC_LUBY_MIS, GC_IS_ALG2, "
                  "GC_JP_ALG4)");
        return GC_ERR_INVALID_ARG;
    }
    GC_CUDA_TRY(cudaSetDevice(g->device));
    if (g->dist) {
        if (ldf) {
            set_error("gc_color_ex: GC_LDF is single-GPU only");
            return GC_ERR_INVALID_ARG;
        }
        return gc_color_dist(g, o, colors_out, stats);
    }

    const bool luby = kind == GC_LUBY_MIS;
    // Alg.2 as written / Alg.2 + Alg.4: COUNT mode only
    const int jpv = kind == GC_IS_ALG2 ? 2 : kind == GC_JP_ALG4 ? 3 : luby ? 1 : 0;
    int mode = o->mode;
    if (jpv >= 2) mode = GC_MODE_COUNT;
    // AUTO: on low-degree graphs (meshes, grids) a colouring takes few rounds
    // and the plain sweep is fastest (measured: 128^3 mesh 0.47 ms sweep vs
    // 0.77 ms event); skewed graphs take thousands of rounds and need the
    // work-efficient event mode (R-MAT s24: 107 ms event vs 1689 ms sweep).
    // Luby-MIS: SWEEP runs Alg.2 + Alg.3 literally; COUNT computes the same
    // colouring (first-fit greedy in decreasing weight order, R10) as a
    // Jones-Plassmann wavefront over predecessor counts -- AUTO takes it.
    // Measured (profiles/r01_configs.jsonl): COUNT wins on ER (0.73 vs 1.83 ms),
    // rgg (0.63 vs 1.33), R-MAT (26.8 vs 1689) and small grids (64^2: 0.10 vs
    // 0.18, one launch); the plain sweep only on large meshes (128^3: 0.48 vs
    // 0.58; 117^3: 0.43 vs 0.47), whose few uniform rounds stream the CSR.
    // Large non-skewed graphs: a round's decrements are random 8-byte atomics
    // over the whole count array, which leaves L2 past ~2^22 vertices; the
    // sweep's status reads win there (rgg_n_2_23: sweep 7.1 vs count 8.4 ms,
    // 2^24: 14.3 vs 29.7; 2^22: count 2.2 vs 3.7 -- profiles/r02_rgg_modes.txt).
    // Skewed graphs (max degree > 8x the mean: power law) take thousands of
    // rounds and keep COUNT at any size.
    const bool skewed = g->n > 0 && g->max_deg > 8 * std::max<int64_t>(1, g->nnz / g->n);
    if (mode == GC_MODE_AUTO)
        mode = (luby || g->n < (1 << 20) || (g->max_deg > 8 && (skewed || g->n <= (1 << 22)))) ? GC_MODE_COUNT
                                                                                                : GC_MODE_SWEEP;
    if (ldf) mode = GC_MODE_COUNT;  // (degree, weight) keys: COUNT kernels only
    if (luby && mode != GC_MODE_COUNT) mode = GC_MODE_SWEEP;
    if (H != 1 && mode != GC_MODE_COUNT) mode = GC_MODE_SWEEP;  // multi-hash: SWEEP or COUNT

    int rc = ensure_scratch(g, mode == GC_MODE_EVENT || mode == GC_MODE_EVENT_MULTI, luby);  // luby: S is also the fallback's
    if (rc) return rc;
    RunParams p;
    p.H = H;
    for (int j = 0; j < H; ++j) p.keys.k[j] = weight_key(o->seed, j);
    p.thread_deg_max = o->thread_deg_max > 0 ? o->thread_deg_max : 8;
    p.hub_deg_min = o->hub_deg_min > 0 ? o->hub_deg_min : 4096;
    p.eval_big_min = o->hub_deg_min > 0 ? o->hub_deg_min : 256;
    p.batch_rounds = o->batch_rounds;
    p.max_rounds = (int64_t)(0x7FFFFFFFll / (2 * H)) + 1;
    p.ldf = ldf;
    Profile prof;
    prof.on = (o->flags & GC_PROFILE) != 0;
    p.prof = &prof;
    if (ldf) {  // the degree of R21 is the number of distinct neighbours
        rc = ensure_strict_rows(g);
        if (rc) return rc;
    }

    EventPair ev;  // destroyed on every exit path
    GC_CUDA_TRY(cudaEventCreate(&ev.e0));
    GC_CUDA_TRY(cudaEventCreate(&ev.e1));
    GC_CUDA_TRY(cudaEventRecord(ev.e0, g->stream));
    cudaEvent_t e0 = ev.e0, e1 = ev.e1;
    RunResult res;
    auto run_count_variant = [&]() {
        if (g->count_unsafe) return (int)GC_ERR_NOT_SYMMETRIC;
        if (jpv >= 1) {
            int rs = ensure_strict_rows(g);
            if (rs) return rs;
            return run_count_jp(g, p, &res, jpv);
        }
        return run_count_maxmin(g, p, &res);
    };
    if (kind == GC_HASH_IS(0)) {
        mode = GC_MODE_SWEEP;  // its own per-round kernels (gc_hash.cu)
        rc = run_hash_is(g, p, GC_VARIANT_HASHES(o->variant), &res);
    } else if (mode == GC_MODE_COUNT)
        rc = run_count_variant();
    else if (luby)
        rc = run_luby(g, p, &res);
    else if (mode == GC_MODE_EVENT)
        rc = run_persistent_maxmin(g, p, &res);
    else if (mode == GC_MODE_EVENT_MULTI)
        rc = run_event_maxmin(g, p, &res);
    else
        rc = run_sweep_maxmin(g, p, &res);
    if (rc == GC_ERR_NOT_SYMMETRIC && mode == GC_MODE_COUNT && !g->deduped && !g->count_unsafe) {
        // The counts need a symmetric adjacency MULTISET; duplicate entries are
        // legal input (adjacency sets decide the colouring).  Switch the handle
        // once to its deduplicated, row-sorted copy and rerun (gc_dedup.cu).
        rc = dedup_csr(g);  // sets g->deduped on success only
        if (!rc) rc = run_count_variant();
        else if (rc == GC_ERR_OOM || rc == GC_ERR_TOO_LARGE) rc = GC_ERR_NOT_SYMMETRIC;  // no copy: fall back
    }
    if (rc == GC_ERR_TOO_LARGE && mode == GC_MODE_COUNT && jpv < 2 && !ldf) {
        // a round's item count overflowed the persistent kernel's round word
        // (gc_count.cu, trap 9): the EVENT / SWEEP kernels have no such field
        g->count_unsafe = true;
        rc = GC_ERR_NOT_SYMMETRIC;
    }
    if (rc == GC_ERR_NOT_SYMMETRIC && mode == GC_MODE_COUNT && jpv < 2 && !ldf) {
        // Still asymmetric after deduplication: the adjacency SETS are not
        // symmetric (a count underflow or a stall -- never a silently wrong
        // colour).  The witness / sweep kernels test the set
        // they are given: rerun there (Alg.2 / Alg.4 have no such fallback).
        g->count_unsafe = true;
        if (luby) {
            mode = GC_MODE_SWEEP;
            rc = run_luby(g, p, &res);
        } else if (H != 1) {
            mode = GC_MODE_SWEEP;
            rc = run_sweep_maxmin(g, p, &res);
        } else {
            mode = GC_MODE_EVENT;
            rc = ensure_scratch(g, true, false);
            if (!rc) rc = run_persistent_maxmin(g, p, &res);
        }
    }
    if (rc) return rc;
    int64_t launches = res.launches;
    int64_t ncol = count_colors_device(g, g->s.C, g->n, (o->flags & GC_COMPACT) != 0, g->s.C,
                                       &launches, res.max_color);
    if (ncol < 0) return ncol;
    if (g->n > 0) {
        GC_CUDA_TRY(cudaMemcpyAsync(colors_out, g->s.C, sizeof(int32_t) * (size_t)g->n,
                                    cudaMemcpyDefault, g->stream));
    }
    GC_CUDA_TRY(cudaEventRecord(e1, g->stream));
    GC_CUDA_TRY(cudaEventSynchronize(e1));
    float ms = 0.f;
    cudaEventElapsedTime(&ms, e0, e1);
    if (!luby && kind != GC_HASH_IS(0) && (o->flags & GC_COMPACT) == 0) {
        // raw colours are < 2RH; they must fit int32 (GC_ERR_TOO_LARGE otherwise)
        if ((uint64_t)2 * (uint64_t)res.rounds * (uint64_t)H > 0x7FFFFFFFull) {
            set_error("colours exceed INT32_MAX; use GC_COMPACT");
            return GC_ERR_TOO_LARGE;
        }
    }
    if (stats) {
        stats->mode_used = mode;
        stats->rounds = res.rounds;
        stats->inner_iterations = res.inner;
        stats->n_colors = ncol;
        stats->launches = launches;
        stats->ms = ms;
        for (int c = 0; c < 4; ++c) {
            stats->kernel_ms[c] = prof.ms[c];
            stats->kernel_launches[c] = prof.launches[c];
            stats->kernel_bytes[c] = prof.bytes[c];
        }
        stats->visits = prof.visits;
        if (stats->launch_us && stats->launch_cap > 0) {
            size_t m = std::min<size_t>((size_t)stats->launch_cap, prof.launch_us.size());
            memcpy(stats->launch_us, prof.launch_us.data(), m * sizeof(float));
        }
        if (prof.on && stats->round_stats && stats->round_stats_cap > 0) {
            int64_t m = std::min<int64_t>(std::min<int64_t>(stats->round_stats_cap, res.rounds + 1),
                                          g->s.nk_cap);
            if (m > 0)
                GC_CUDA_TRY(cudaMemcpy(stats->round_stats, g->s.rstat, sizeof(int64_t) * 16 * m,
                                       cudaMemcpyDeviceToHost));
        }
        // (Hash IS keeps no per-round frontier trace: its entries are left untouched)
        if (stats->frontier_sizes && stats->frontier_cap > 0 && !luby && kind != GC_HASH_IS(0)) {
            int64_t m = std::min<int64_t>(std::min<int64_t>(stats->frontier_cap, res.rounds),
                                          g->s.nk_cap);
            if (m > 0)
                GC_CUDA_TRY(cudaMemcpy(stats->frontier_sizes, g->s.nk, sizeof(int64_t) * m,
                                       cudaMemcpyDefault));
        }
    }
    return ncol;
}

int64_t gc_color(gc_graph *g, uint64_t seed, int32_t variant, int32_t *colors_out) {
    gc_options o;
    memset(&o, 0, sizeof(o));
    o.struct_size = sizeof(o);
    o.variant = variant;
    o.seed = seed;
    return gc_color_ex(g, &o, colors_out, nullptr);
}

int gc_priorities(uint64_t seed, int32_t j, int64_t v_begin, int64_t count, uint32_t *out) {
    if (count < 0 || v_begin < 0 || (count > 0 && !out) || j < 0 || j >= GC_MAX_HASHES) {
        set_error("gc_priorities: bad arguments");
        return GC_ERR_INVALID_ARG;
    }
    int dev = 0, sms = 0;
    int rc = current_device_ok(&dev, &sms);
    if (rc) return rc;
    if (count == 0) return GC_OK;
    if (is_device_ptr(out)) {
        rc = launch_priorities(seed, j, v_begin, count, out, 0);
        if (rc) return rc;
        GC_CUDA_TRY(cudaStreamSynchronize(0));
        return GC_OK;
    }
    uint32_t *d = nullptr;
    GC_CUDA_TRY(dmalloc(&d, sizeof(uint32_t) * (size_t)count));
    rc = launch_priorities(seed, j, v_begin, count, d, 0);
    if (!rc) {
        cudaError_t e = cudaMemcpy(out, d, sizeof(uint32_t) * (size_t)count, cudaMemcpyDeviceToHost);
        if (e != cudaSuccess) rc = cuda_fail(e, "gc_priorities copy");
    }
    dfree(d);
    return rc;
}

int64_t gc_count_colors(const int32_t *colors, int64_t n) {
    if (n < 0 || (n > 0 && !colors)) {
        set_error("gc_count_colors: bad arguments");
        return GC_ERR_INVALID_ARG;
    }
    if (n == 0) return 0;
    int dev = 0, sms = 0;
    int rc = current_device_ok(&dev, &sms);
    if (rc) return rc;
    gc_graph tmp;
    tmp.device = dev;
    tmp.sm_count = sms;
    tmp.n = n;
    const uint32_t *C = reinterpret_cast<const uint32_t *>(colors);
    uint32_t *dC = nullptr;
    if (!is_device_ptr(colors)) {
        GC_CUDA_TRY(dmalloc(&dC, sizeof(uint32_t) * (size_t)n));
        GC_CUDA_TRY(cudaMemcpy(dC, colors, sizeof(uint32_t) * (size_t)n, cudaMemcpyHostToDevice));
        C = dC;
    }
    int64_t launches = 0;
    int64_t r = GC_OK;
    cudaError_t e = dmalloc(&tmp.s.ctr, kCtrWords * sizeof(unsigned long long));
    if (e == cudaSuccess) e = hmalloc(&tmp.s.host_pinned, 4096);
    if (e != cudaSuccess) r = cuda_fail(e, "gc_count_colors alloc");
    if (r == GC_OK) r = count_colors_device(&tmp, C, n, false, nullptr, &launches);
    free_scratch(tmp.s);
    dfree(dC);
    return r;
}

}  // extern "C"
