// srad_reduce.cu — the per-iteration statistic of a full SRAD iteration
// (A27): q0^2 = var(I) / mean(I)^2 over the image.
//
// fp64 (sum, sum of squares) partials with a fixed grid and a fixed
// combination order, so the value is reproducible run to run (and therefore so
// is every SRAD iterate).  Only the FIRST iteration of a chain reads I for it
// (k_sum2); the fused SRAD pass (K1S) emits the statistics of the image it
// writes as one partial per CTA, so later iterations reduce those few hundred
// partials at the start of their own pass (srad_q0_from_partials in
// kernel_tile2d.cu) and never re-read the image.  k_q0 turns partials into
// SRAD1's constants {q0, q0/(1+q0), 1/(q0(1+q0))} for the generic kernel (K0).
//
// Workspace: [cap] double2 partials A | [cap] double2 partials B | 3 floats.
#include <cuda_runtime.h>

#include "launch.hpp"
#include "ops.cuh"

namespace lift {
namespace {

constexpr int kThreads = 256;
constexpr int kUnroll = 4;     // float4 loads in flight per thread per iteration

int n_blocks(int num_sms) { return num_sms * 4; }

__global__ void __launch_bounds__(kThreads) k_sum2(const float* __restrict__ x, int64_t n, double2* partials) {
  pdl_launch_dependents();
  pdl_wait();
  double s = 0.0, ss = 0.0;
  const int64_t n4 = n / 4;
  const float4* x4 = reinterpret_cast<const float4*>(x);
  const bool vec = (reinterpret_cast<uintptr_t>(x) & 15u) == 0;
  const int64_t stride = (int64_t)gridDim.x * blockDim.x;
  const int64_t t0 = (int64_t)blockIdx.x * blockDim.x + threadIdx.x;
  auto add = [&](float v) {
    const double d = v;
    s += d;
    ss = fma(d, d, ss);
  };
  int64_t tail = 0;
  if (vec) {
    int64_t i = t0;
    // kUnroll independent 16-B loads in flight, then accumulate in index order
    for (; i + (kUnroll - 1) * stride < n4; i += kUnroll * stride) {
      float4 v[kUnroll];
#pragma unroll
      for (int u = 0; u < kUnroll; ++u) v[u] = __ldg(x4 + i + u * stride);
#pragma unroll
      for (int u = 0; u < kUnroll; ++u) {
        add(v[u].x);
        add(v[u].y);
        add(v[u].z);
        add(v[u].w);
      }
    }
    for (; i < n4; i += stride) {
      const float4 v = __ldg(x4 + i);
      add(v.x);
      add(v.y);
      add(v.z);
      add(v.w);
    }
    tail = 4 * n4;
  }
  for (int64_t i = tail + t0; i < n; i += stride) add(__ldg(x + i));
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
  pdl_launch_dependents();
  pdl_wait();
  double s = 0.0, ss = 0.0;
  for (int i = threadIdx.x; i < nb; i += 32) {
    s += partials[i].x;
    ss += partials[i].y;
  }
  for (int o = 16; o > 0; o >>= 1) {
    s += __shfl_down_sync(0xffffffffu, s, o);
    ss += __shfl_down_sync(0xffffffffu, ss, o);
  }
  if (threadIdx.x == 0) srad1_constants(srad_q0sqr(s, ss, n), out3);
}

}  // namespace

int srad_partials_cap(int num_sms) { return num_sms * 8; }

size_t srad_workspace_bytes(int num_sms) { return 2 * (size_t)srad_partials_cap(num_sms) * sizeof(double2) + 64; }

double2* srad_partials_ptr(void* ws, int num_sms, int which) {
  return reinterpret_cast<double2*>(ws) + (size_t)which * srad_partials_cap(num_sms);
}

const float* srad_q0_ptr(void* ws, int num_sms) {
  return reinterpret_cast<const float*>(srad_partials_ptr(ws, num_sms, 2));
}

cudaError_t launch_srad_partials(const float* img, int64_t n, double2* partials, int num_sms, cudaStream_t stream,
                                 int* nparts) {
  const int nb = n_blocks(num_sms);
  void* args[] = {(void*)&img, (void*)&n, (void*)&partials};
  *nparts = nb;
  return launch_kernel(reinterpret_cast<const void*>(k_sum2), dim3(nb), dim3(kThreads), args, 0, stream, true);
}

cudaError_t launch_srad_q0(const float* img, int64_t n, void* ws, int num_sms, cudaStream_t stream) {
  double2* partials = srad_partials_ptr(ws, num_sms, 0);
  float* out3 = const_cast<float*>(srad_q0_ptr(ws, num_sms));
  int nb = 0;
  cudaError_t e = launch_srad_partials(img, n, partials, num_sms, stream, &nb);
  if (e != cudaSuccess) return e;
  void* args[] = {(void*)&partials, (void*)&nb, (void*)&n, (void*)&out3};
  return launch_kernel(reinterpret_cast<const void*>(k_q0), dim3(1), dim3(32), args, 0, stream, true);
}

}  // namespace lift
