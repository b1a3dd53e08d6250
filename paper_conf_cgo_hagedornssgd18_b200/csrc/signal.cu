// signal.cu — the waiting side of the fused halo put (slab mode, multi-GPU).
//
// A one-thread kernel spins (acquire, system scope) until every flag holds a
// value >= the step number; launched on the compute stream before a step's
// boundary-plane kernel, it orders that kernel's ghost reads after the
// neighbours' peer stores (which their boundary kernel published with a
// release store of the same step number).  Step numbers only grow, so there
// is no ABA.
#include <cuda_runtime.h>

#include "launch.hpp"
#include "tma.cuh"

namespace lift {
namespace {

__global__ void k_wait_signals(const unsigned int* __restrict__ a, const unsigned int* __restrict__ b,
                               unsigned int value) {
  if (a)
    while ((int)(ld_acquire_sys(a) - value) < 0) __nanosleep(64);
  if (b)
    while ((int)(ld_acquire_sys(b) - value) < 0) __nanosleep(64);
}

}  // namespace

cudaError_t launch_wait_signals(const unsigned int* a, const unsigned int* b, unsigned int value,
                                cudaStream_t stream) {
  k_wait_signals<<<1, 1, 0, stream>>>(a, b, value);
  return cudaGetLastError();
}

}  // namespace lift
