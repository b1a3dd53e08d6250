// srad_reduce.cu — the per-iteration statistic of a full SRAD iteration
// (A27): q0^2 = var(I) / mean(I)^2 over the image.
//
// Two passes, fp64, fixed grid and fixed combination order, so the value is
// reproducible run to run (and therefore so is every SRAD iterate): pass 1
// has each CTA accumulate a grid-stride slice (sum, sum of squares) and write
// its partial; pass 2 (one warp) adds the partials in a fixed order and writes
// SRAD1's constants {q0, q0/(1+q0), 1/(q0(1+q0))} for the stencil launch.
#include <cuda_runtime.h>

#include "launch.hpp"
#include "ops.cuh"

namespace lift {
namespace {

constexpr int kThreads = 256;

int n_blocks(int num_sms) { return num_sms * 4; }

__global__ void __launch_bounds__(kThreads) k_sum2(const float* __restrict__ x, int64_t n, double2* partials) {
  double s = 0.0, ss = 0.0;
  const int64_t n4 = n / 4;
  const float4* x4 = reinterpret_cast<const float4*>(x);
  const bool vec = (reinterpret_cast<uintptr_t>(x) & 15u) == 0;
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  if (vec) {
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n4; i += stride) {
      const float4 v = __ldg(x4 + i);
      s += (double)v.x + (double)v.y + (double)v.z + (double)v.w;
      ss += (double)v.x * v.x + (double)v.y * v.y + (double)v.z * v.z + (double)v.w * v.w;
    }
    for (int64_t i = 4 * n4 + (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
      const double v = __ldg(x + i);
      s += v;
      ss += v * v;
    }
  } else {
    for (int64_t i = (int64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
      const double v = __ldg(x + i);
      s += v;
      ss += v * v;
    }
  }
  for (int o = 16; o > 0; o >>= 1) {
    s += __shfl_down_sync(0xffffffffu, s, o);
    ss += __shfl_down_sync(0xffffffffu, ss, o);
  }
  __shared__ double2 red[kThreads / 32];
  if ((threadIdx.x & 31) == 0) red[threadIdx.x >> 5] = make_double2(s, ss);
  __syncthreads();
  if (threadIdx.x == 0) {
    double a = 0.0, b = 0.0;
    for (int w = 0; w < kThreads / 32; ++w) {
      a += red[w].x;
      b += red[w].y;
    }
    partials[blockIdx.x] = make_double2(a, b);
  }
}

__global__ void k_q0(const double2* __restrict__ partials, int nb, int64_t n, float* out3) {
  double s = 0.0, ss = 0.0;
  for (int i = threadIdx.x; i < nb; i += 32) {
    s += partials[i].x;
    ss += partials[i].y;
  }
  for (int o = 16; o > 0; o >>= 1) {
    s += __shfl_down_sync(0xffffffffu, s, o);
    ss += __shfl_down_sync(0xffffffffu, ss, o);
  }
  if (threadIdx.x == 0) {
    const double mean = s / (double)n;
    const double var = ss / (double)n - mean * mean;
    srad1_constants((float)(var / (mean * mean)), out3);
  }
}

}  // namespace

size_t srad_workspace_bytes(int num_sms) { return (size_t)n_blocks(num_sms) * sizeof(double2) + 64; }

const float* srad_q0_ptr(void* ws, int num_sms) {
  return reinterpret_cast<const float*>(reinterpret_cast<char*>(ws) + (size_t)n_blocks(num_sms) * sizeof(double2));
}

cudaError_t launch_srad_q0(const float* img, int64_t n, void* ws, int num_sms, cudaStream_t stream) {
  const int nb = n_blocks(num_sms);
  double2* partials = reinterpret_cast<double2*>(ws);
  float* out3 = const_cast<float*>(srad_q0_ptr(ws, num_sms));
  k_sum2<<<nb, kThreads, 0, stream>>>(img, n, partials);
  k_q0<<<1, 32, 0, stream>>>(partials, nb, n, out3);
  return cudaGetLastError();
}

}  // namespace lift
