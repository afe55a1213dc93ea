// prune_f32.cu -- instantiates the pruning kernels for FP32 partials, F81 (Eq. 20).
#include "prune_kernels.cuh"

namespace mpcgs {
template cudaError_t launch_prune_typed<float, false>(PruneArgs, int, int, cudaStream_t, int&);
}  // namespace mpcgs
