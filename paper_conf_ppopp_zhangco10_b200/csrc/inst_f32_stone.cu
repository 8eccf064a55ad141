// Kernel instantiations of libtridiag.so for T = float, inner = STONE (the
// overflow-free LU-form recursive doubling, NEXT f3).
#include "launch.cuh"

namespace tdg_host {
template cudaError_t dispatch_t<float, tdg::kSTONE>(const void*, const void*, const void*,
                                                const void*, void*, int64_t, int64_t, int,
                                                cudaStream_t, int, int64_t, Layout);
}  // namespace tdg_host
