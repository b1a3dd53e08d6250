// kernel_persist3d.cu — K4: iterate(in, f, n) of a small 3D radius-1
// star stencil (7-point weighted, Hotspot3D) as ONE persistent launch.
// Opt-in (LIFT_K4=1): on B200 it measured slower than one K2 launch per step
// replayed from a CUDA graph (Hotspot3D 8x512x512 x100: 267 vs 303 Gpts/s;
// the taps come from L2 without the shared-memory reuse of K2's TMA boxes,
// and the grid barrier costs about what the launch hand-off does).
//
// A grid that fits in L2 (Rodinia's Hotspot3D is 8 x 512 x 512: 24 MiB per
// step with its power grid) makes every time step latency-bound: ~2 M points
// are a few microseconds of L2 traffic, and a kernel launch per step — even
// graph-replayed with programmatic dependent launch — costs as much again in
// ramp-up, tail and the dependency hand-off.  K4 keeps every CTA resident
// (cooperative launch: co-residency is guaranteed or the launch fails) and
// runs all n steps in one launch, with a grid barrier between steps.  Each
// thread owns float4 output groups (4 consecutive x) in a grid-stride loop;
// the 7 taps come straight from L2 (ld.global.cg: the state written by other
// CTAs in the previous step must not be read through a stale L1 line), the
// point-wise grid (Hotspot P, fixed) through the read-only path.  f is the
// same ops.cuh function with the same tap order as K0/K2, so each step's bits
// equal a K2 step's.  pad is index remapping of the edge taps,
// as in K0.
#include <cuda_runtime.h>

#include <algorithm>
#include <atomic>
#include <cstdlib>
#include <mutex>
#include <string>

#include "common.cuh"
#include "launch.hpp"
#include "ops.cuh"
#include "slots.cuh"

namespace lift {
namespace {

constexpr int kThreads = 512;
// grid-barrier state, one slot per running launch (slots.cuh): c[0]
// arrivals, c[1] generation, c[2] exits (reset by the last CTA)
__device__ LaunchSlot g_launch[kLaunchSlots];

enum K4Op { K4_WSTAR = 0, K4_HOTSPOT = 1 };

__device__ __forceinline__ float4 ldcg4(const float* p) { return __ldcg(reinterpret_cast<const float4*>(p)); }

// neighbour index i (= c - 1 or c + 1) along a dimension of extent n with
// boundary kind k: the in-grid index, or -1 for the constant (pad)
__device__ __forceinline__ int64_t nb_index(int64_t i, int64_t n, int k) {
  if (i >= 0 && i < n) return i;
  if (k == PAD_CONSTANT) return -1;
  return pad_remap(i, n, k);
}

// the 7-point window of 4 consecutive outputs
struct Star4 {
  float x[6];                 // centre row, x offsets -1 .. 4
  float ym[4], yp[4], zm[4], zp[4];
};

template <int I>
struct Star4Acc {
  const Star4& w;
  template <int DZ, int DY, int DX>
  __device__ __forceinline__ float at() const {
    static_assert((DZ != 0) + (DY != 0) + (DX != 0) <= 1, "star access only");
    if constexpr (DZ < 0) return w.zm[I];
    else if constexpr (DZ > 0) return w.zp[I];
    else if constexpr (DY < 0) return w.ym[I];
    else if constexpr (DY > 0) return w.yp[I];
    else return w.x[I + 1 + DX];
  }
};

__device__ __forceinline__ void set4(float (&d)[4], float4 v) {
  d[0] = v.x; d[1] = v.y; d[2] = v.z; d[3] = v.w;
}

template <int OP>
__device__ __forceinline__ float4 eval4(const StencilParams& p, const Star4& w, float4 pw) {
  const float pv[4] = {pw.x, pw.y, pw.z, pw.w};
  float v[4];
  static_for<4>([&](auto II) {
    constexpr int i = decltype(II)::value;
    if constexpr (OP == K4_WSTAR) v[i] = op_weighted<1, 1, 1, true>(Star4Acc<i>{w}, p.wbox);
    else v[i] = op_hotspot3d(Star4Acc<i>{w}, pv[i], p.prm);
  });
  return make_float4(v[0], v[1], v[2], v[3]);
}

// A unit is a column of ZB planes of one float4 group (4 consecutive x) of
// one row; lanes of a warp hold consecutive groups, so the x-halo taps come
// from the neighbouring lanes by shuffles and each plane's centre row is
// loaded once and reused as the z-1 / z+1 taps of the next / previous plane.
template <int OP, int ZB>
__global__ void __launch_bounds__(kThreads) k4_iterate(const __grid_constant__ StencilParams p, float* s0, float* s1,
                                                       const float* __restrict__ aux, int n_steps) {
  const int64_t nx = p.n[2], ny = p.n[1], nz = p.n[0];
  const uint32_t nx4 = (uint32_t)(nx >> 2);
  const uint32_t nzb = (uint32_t)((nz + ZB - 1) / ZB);
  const uint32_t units = (uint32_t)ny * nx4 * nzb;
  const uint32_t wstride = gridDim.x * blockDim.x;
  const int lane = threadIdx.x & 31;
  const int kx = p.kind[2];
  const float4 cv = make_float4(p.pad_value, p.pad_value, p.pad_value, p.pad_value);
  const float* in = s0;
  float* out = s1;
  int slot = 0;                      // used by thread 0 only
  if (threadIdx.x == 0 && n_steps > 1) slot = claim_launch_slot(g_launch);
  for (int t = 0; t < n_steps; ++t) {
    // warp-uniform loop (full-warp shuffles); units < 2^31 (L2-resident grids only)
    for (uint32_t u0 = blockIdx.x * blockDim.x + (threadIdx.x & ~31u); u0 < units; u0 += wstride) {
      const uint32_t u = u0 + lane;
      const bool ok = u < units;
      const uint32_t uu = ok ? u : units - 1;
      const uint32_t r = uu / nx4;
      const uint32_t xq = uu - r * nx4;
      const uint32_t zb = r / (uint32_t)ny;
      const int64_t y = r - zb * (uint32_t)ny;
      const int64_t x0 = (int64_t)xq * 4;
      const int64_t z0 = (int64_t)zb * ZB;
      const int64_t ym = nb_index(y - 1, ny, p.kind[1]), yp = nb_index(y + 1, ny, p.kind[1]);
      // x halo from the neighbouring lanes when they hold the adjacent group of the same row
      const bool lnb = lane > 0 && xq > 0;
      const bool rnb = lane < 31 && xq + 1 < nx4 && u + 1 < units;
      const int64_t xl = nb_index(x0 - 1, nx, kx), xr = nb_index(x0 + 4, nx, kx);
      auto row_at = [&](int64_t zz, int64_t yy) -> int64_t { return (zz * ny + yy) * nx; };
      auto plane = [&](int64_t zz) -> float4 {      // centre group of plane zz (padded index)
        const int64_t zi = nb_index(zz, nz, p.kind[0]);
        return zi < 0 ? cv : ldcg4(in + row_at(zi, y) + x0);
      };
      float4 cm = plane(z0 - 1), cc = plane(z0);
      const int zn = (int)(nz - z0 < ZB ? nz - z0 : ZB);
#pragma unroll
      for (int k = 0; k < ZB; ++k) {
        {   // every lane runs all ZB planes (full-warp shuffles); planes past the grid are not stored
          const bool kv = k < zn;
          const int64_t z = kv ? z0 + k : nz - 1;
          const float4 cp = plane(z + 1);
          Star4 w;
          w.x[1] = cc.x; w.x[2] = cc.y; w.x[3] = cc.z; w.x[4] = cc.w;
          const float l = __shfl_up_sync(0xffffffffu, cc.w, 1);
          const float rr = __shfl_down_sync(0xffffffffu, cc.x, 1);
          const int64_t rb = row_at(z, y);
          w.x[0] = lnb ? l : (xl < 0 ? p.pad_value : __ldcg(in + rb + xl));
          w.x[5] = rnb ? rr : (xr < 0 ? p.pad_value : __ldcg(in + rb + xr));
          set4(w.zm, cm);
          set4(w.zp, cp);
          set4(w.ym, ym < 0 ? cv : ldcg4(in + row_at(z, ym) + x0));
          set4(w.yp, yp < 0 ? cv : ldcg4(in + row_at(z, yp) + x0));
          float4 pw = make_float4(0.f, 0.f, 0.f, 0.f);
          if constexpr (OP == K4_HOTSPOT) pw = __ldg(reinterpret_cast<const float4*>(aux + rb + x0));
          const float4 v = eval4<OP>(p, w, pw);
          if (ok && kv) *reinterpret_cast<float4*>(out + rb + x0) = v;
          cm = cc;
          cc = cp;
        }
      }
    }
    if (t + 1 < n_steps) {
      // grid barrier (all CTAs are co-resident): arrive, the last arriver
      // bumps the generation, everyone waits for it
      __syncthreads();
      if (threadIdx.x == 0) {
        __threadfence();
        const unsigned int a = atomicAdd(&g_launch[slot].c[0], 1u);
        if (a == (unsigned)(t + 1) * gridDim.x - 1) {
          __threadfence();
          atomicExch(&g_launch[slot].c[1], (unsigned)(t + 1));
        } else {
          while (*reinterpret_cast<volatile unsigned int*>(&g_launch[slot].c[1]) < (unsigned)(t + 1)) __nanosleep(20);
        }
        __threadfence();
      }
      __syncthreads();
    }
    const float* nin = out;
    out = const_cast<float*>(in);
    in = nin;
  }
  // the last CTA out resets the slot (every CTA has passed every barrier by then)
  if (threadIdx.x == 0 && n_steps > 1) {
    if (atomicAdd(&g_launch[slot].c[2], 1u) == gridDim.x - 1) release_launch_slot(g_launch, slot);
  }
}

struct Launcher {
  const void* fn;
  int blocks_per_sm;
};

template <int OP, int ZB>
Launcher get_launcher() {
  static Launcher L{};
  static std::once_flag once;
  std::call_once(once, [] {
    auto fn = k4_iterate<OP, ZB>;
    int occ = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, fn, kThreads, 0) != cudaSuccess) occ = 0;
    cudaGetLastError();
    L = Launcher{reinterpret_cast<const void*>(fn), occ};
  });
  return L;
}

}  // namespace

bool persist3d_supported(const StencilParams& p, const float* s0, const float* s1, const float* aux) {
  // opt-in (LIFT_K4=1): measured slower than graph-replayed K2 steps on
  // Hotspot3D 8x512x512 (267 vs 303 Gpts/s)
  const char* e = getenv("LIFT_K4");
  if (!(e && e[0] == '1')) return false;
  if (p.slab || p.n[0] < 1 || has_dampen(p)) return false;
  if (p.op != OP_WEIGHTED && p.op != OP_HOTSPOT3D) return false;
  for (int d = 0; d < 3; ++d)
    if (p.size[d] != 3 || p.lo[d] != 1 || p.hi[d] != 1 || p.step[d] != 1) return false;
  if (p.op == OP_WEIGHTED) {
    for (int k = 0; k < 27; ++k) {
      const int kz = k / 9, ky = (k / 3) % 3, kx = k % 3;
      if ((kz != 1) + (ky != 1) + (kx != 1) > 1 && p.wbox[k] != 0.0f) return false;   // star only
    }
  }
  if (p.n[2] % 4 != 0) return false;
  auto al = [](const void* q) { return (reinterpret_cast<uintptr_t>(q) & 15u) == 0; };
  if (!al(s0) || !al(s1) || (aux && !al(aux))) return false;
  // L2-resident grids only (state ping-pong + the point-wise grid within
  // half the 126 MB L2); larger grids are HBM-bound and run on K2
  const int64_t pts = p.n[0] * p.n[1] * p.n[2];
  const int64_t bytes = pts * 4 * (p.op == OP_HOTSPOT3D ? 3 : 2);
  return bytes <= (64ll << 20);
}

cudaError_t launch_persist3d(const StencilParams& p, float* s0, float* s1, const float* aux, int n_steps,
                             cudaStream_t stream, int num_sms, std::string* err) {
  const char* ez = getenv("LIFT_K4_ZB");
  const int zbv = ez ? atoi(ez) : 4;
  Launcher L;
  if (zbv == 2) L = p.op == OP_HOTSPOT3D ? get_launcher<K4_HOTSPOT, 2>() : get_launcher<K4_WSTAR, 2>();
  else if (zbv == 8) L = p.op == OP_HOTSPOT3D ? get_launcher<K4_HOTSPOT, 8>() : get_launcher<K4_WSTAR, 8>();
  else L = p.op == OP_HOTSPOT3D ? get_launcher<K4_HOTSPOT, 4>() : get_launcher<K4_WSTAR, 4>();
  if (L.blocks_per_sm < 1) {
    *err = "K4: kernel cannot be resident";
    return cudaErrorInvalidConfiguration;
  }
  const int64_t units = ((p.n[0] + zbv - 1) / zbv) * p.n[1] * (p.n[2] / 4);
  int64_t grid = (int64_t)num_sms * L.blocks_per_sm;
  const int64_t need = (units + kThreads - 1) / kThreads;
  if (grid > need) grid = need;
  void* args[] = {(void*)&p, (void*)&s0, (void*)&s1, (void*)&aux, (void*)&n_steps};
  // cooperative attribute: all CTAs co-resident or the launch fails (never a
  // silent deadlock in the grid barrier); capturable into CUDA graphs
  cudaLaunchConfig_t cfg{};
  cfg.gridDim = dim3((unsigned)grid);
  cfg.blockDim = dim3(kThreads);
  cfg.dynamicSmemBytes = 0;
  cfg.stream = stream;
  cudaLaunchAttribute at[1];
  at[0].id = cudaLaunchAttributeCooperative;
  at[0].val.cooperative = 1;
  cfg.attrs = at;
  cfg.numAttrs = 1;
  set_last_kernel("k4_iterate");
  return cudaLaunchKernelExC(&cfg, L.fn, args);
}

}  // namespace lift
