// Kernel instantiations of libtridiag.so for T = double, inner = PCR
// (one translation unit per combination so nvcc builds them in parallel).
#include "launch.cuh"

namespace tdg_host {
template cudaError_t dispatch_t<double, tdg::kPCR>(const void*, const void*, const void*, const void*,
                                            void*, int64_t, int64_t, int, cudaStream_t, int,
                                            int64_t, Layout);
}  // namespace tdg_host
