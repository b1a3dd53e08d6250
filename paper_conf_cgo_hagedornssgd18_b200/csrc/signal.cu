// signal.cu — the waiting side of the fused halo put (slab mode, multi-GPU).
//
// A one-thread kernel spins (acquire, system scope) until every flag holds a
// value >= the step number; launched on the compute stream before a step's
// boundary-plane kernel, it orders that kernel's ghost reads after the
// neighbours' peer stores (which their boundary kernel published with a
// release store of the same step number).  Step numbers only grow, so there
// is no ABA.  The wait is bounded (stencil_set_wait_timeout_ms): a flag that
// never arrives is reported through stencil_device_fault, not a hang.
#include <cuda_runtime.h>

#include "launch.hpp"
#include "tma.cuh"

namespace lift {
namespace {

__global__ void k_wait_signals(const unsigned int* __restrict__ a, const unsigned int* __restrict__ b,
                               unsigned int value, unsigned long long timeout_ns, unsigned int* fault) {
  // bounded (tma.cuh): a neighbour that never signals records a fault
  // instead of hanging the stream
  if (a) spin_until_bounded(a, value, timeout_ns, fault, kFaultWaitLo);
  if (b) spin_until_bounded(b, value, timeout_ns, fault, kFaultWaitHi);
}

}  // namespace

cudaError_t launch_wait_signals(const unsigned int* a, const unsigned int* b, unsigned int value,
                                unsigned long long timeout_ns, unsigned int* fault, cudaStream_t stream) {
  k_wait_signals<<<1, 1, 0, stream>>>(a, b, value, timeout_ns, fault);
  return cudaGetLastError();
}

}  // namespace lift
