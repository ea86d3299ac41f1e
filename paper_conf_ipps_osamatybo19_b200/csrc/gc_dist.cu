// gc_dist.cu -- 1D vertex-range partition across GPUs.
#include "gc_internal.cuh"

namespace gc {
void destroy_dist(gc_graph *g) { (void)g; }
}  // namespace gc

using namespace gc;

extern "C" {

int64_t gc_color_dist(gc_graph *g, const gc_options *o, int32_t *colors_out, gc_stats *stats) {
    (void)g; (void)o; (void)colors_out; (void)stats;
    set_error("distributed colouring not implemented yet");
    return GC_ERR_INVALID_ARG;
}

int gc_create_csr_dist(int64_t, int64_t, int64_t, int64_t, const int64_t *, const uint32_t *,
                       const void *, int, int, uint32_t, gc_graph **out) {
    if (out) *out = nullptr;
    set_error("distributed colouring not implemented yet");
    return GC_ERR_INVALID_ARG;
}

int gc_nccl_unique_id(void *) {
    set_error("distributed colouring not implemented yet");
    return GC_ERR_INVALID_ARG;
}

}  // extern "C"
