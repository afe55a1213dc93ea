// prune_f32_gm.cu -- instantiates the pruning kernels for FP32 partials, general reversible model (F84 / HKY85).
#include "prune_kernels.cuh"

namespace mpcgs {
template cudaError_t launch_prune_typed<float, true>(PruneArgs, int, int, cudaStream_t, int&);
}  // namespace mpcgs
