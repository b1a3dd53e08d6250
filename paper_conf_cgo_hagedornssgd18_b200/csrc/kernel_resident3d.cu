// kernel_resident3d.cu — K6: iterate(in, f, n) of a small 3D grid
// with the whole grid resident in shared memory across all n steps.
//
// B200 has 148 x 227 KB of shared memory — 33 MB on chip, more than a few-
// plane grid like Hotspot3D's 512 x 512 x 8 (8 MB state + 8 MB power map).
// K6 is ONE cooperative launch: every CTA owns a 128 x TY (x, y) tile over
// all nz planes (the K2C column) and keeps it in shared memory for the whole
// iteration, in two boxes (ping-pong, each with a one-cell halo ring) plus
// the tile of the point-wise grid.  A time step is
//   compute box[t+1] from box[t] (ops.cuh f, the same sequence as every
//     other kernel family, so the result is bitwise that of n K2 sweeps);
//   store the tile's edge cells (the cells its neighbours read) to global
//     memory (the state buffer of that step);
//   raise this tile's step flag, wait for the flags of the (<= 4) tiles
//     whose edges fill its halo (point-to-point, no grid barrier);
//   refill box[t+1]'s halo ring: in-grid cells from global (L2, written by
//     the neighbour tiles just before the barrier), out-of-grid cells by pad
//     (P:407-466): the constant, or the remapped cell — from this tile's box
//     when it lies in it (clamp / mirror / reflect), else from global (wrap).
// Only the last step writes the whole tile to HBM.  Per step the traffic is
// the halo rings (~9 KB per CTA) instead of the grid (24 MB): the launch
// overhead and the DRAM/L2 round trips of n separate sweeps disappear.
// The step flags are the launch's own slot (claimed by grid id, slots.cuh).
#include <cuda.h>
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdint>
#include <cstdlib>
#include <mutex>
#include <string>

#include "colwin.cuh"
#include "common.cuh"
#include "launch.hpp"
#include "slots.cuh"
#include "tma.cuh"

namespace lift {
namespace {

constexpr int TX = 128;
constexpr int XH = 4;
constexpr int BX = TX + 2 * XH;
constexpr int NW = 16;
constexpr int NT = NW * 32;
constexpr int kMaxNz = 16;
constexpr int kMaxTiles = 256;
constexpr int kSlots = 4096;

// per running launch: owner, exit counter, and one step flag per tile
struct K6Slot {
  unsigned long long owner;
  unsigned int exits;
  unsigned int pad_;
  unsigned int flag[kMaxTiles];
};
__device__ K6Slot g_k6[kSlots];

struct Geo {
  int nz, ny, nx, x0, y0, hv, wv;
};

// The ring cells just outside the tile's valid region (a star stencil never
// reads the corners), cell q in [0, 2*wv + 2*hv): its box row and column.
__device__ __forceinline__ void ring_cell(const Geo& G, int q, bool inner, int& r, int& col) {
  if (q < 2 * G.wv) {
    r = q < G.wv ? (inner ? 1 : 0) : (inner ? G.hv : G.hv + 1);
    col = XH + (q < G.wv ? q : q - G.wv);
  } else {
    const int q2 = q - 2 * G.wv;
    col = q2 < G.hv ? (inner ? XH : XH - 1) : (inner ? XH + G.wv - 1 : XH + G.wv);
    r = 1 + (q2 < G.hv ? q2 : q2 - G.hv);
  }
}

// Refill the halo ring of ``box`` for the state whose in-grid cells are in
// ``g`` (global): thread q < 2wv + 2hv owns ring cell q in every plane (one
// address computation, nz independent loads, then the stores; the sources
// are valid cells, never ring cells).
template <int BY>
__device__ __forceinline__ void fill_halo(const StencilParams& p, const Geo& G, float* box, const float* g, int tid) {
  const int per = 2 * G.wv + 2 * G.hv;
  if (tid >= per) return;
  int r, col;
  ring_cell(G, tid, false, r, col);
  int gy = G.y0 - 1 + r, gx = G.x0 - XH + col;
  const bool oy = gy < 0 || gy >= G.ny, ox = gx < 0 || gx >= G.nx;
  const int kx = p.kind[2], ky = p.kind[1];
  int mode;            // 0: constant, 1: own box, 2: global
  int src = 0;
  int64_t goff = 0;
  if ((oy && ky == PAD_CONSTANT) || (ox && kx == PAD_CONSTANT)) {
    mode = 0;
  } else {
    if (oy) gy = (int)pad_remap(gy, G.ny, ky);
    if (ox) gx = (int)pad_remap(gx, G.nx, kx);
    const int br = gy - (G.y0 - 1), bc = gx - (G.x0 - XH);
    if (br >= 1 && br <= G.hv && bc >= XH && bc < XH + G.wv) {
      mode = 1;
      src = br * BX + bc;
    } else {
      mode = 2;
      goff = (int64_t)gy * G.nx + gx;
    }
  }
  const int64_t gplane = (int64_t)G.ny * G.nx;
  const int dst = r * BX + col;
  float v[kMaxNz];
#pragma unroll
  for (int z = 0; z < kMaxNz; ++z)
    if (z < G.nz)
      v[z] = mode == 0 ? p.pad_value : (mode == 1 ? box[z * BY * BX + src] : __ldcg(g + z * gplane + goff));
#pragma unroll
  for (int z = 0; z < kMaxNz; ++z)
    if (z < G.nz) box[z * BY * BX + dst] = v[z];
}

// the tile's valid edge cells (rows y0, y0+hv-1; columns x0, x0+wv-1) to global
template <int BY>
__device__ __forceinline__ void store_edges(const Geo& G, const float* box, float* g, int tid) {
  const int per = 2 * G.wv + 2 * G.hv;
  if (tid >= per) return;
  int r, col;
  ring_cell(G, tid, true, r, col);
  const int64_t goff = (int64_t)(G.y0 - 1 + r) * G.nx + (G.x0 - XH + col);
  const int64_t gplane = (int64_t)G.ny * G.nx;
#pragma unroll
  for (int z = 0; z < kMaxNz; ++z)
    if (z < G.nz) __stcg(g + z * gplane + goff, box[z * BY * BX + r * BX + col]);
}

__device__ __forceinline__ void st_release_gpu(unsigned int* p, unsigned int v) {
  asm volatile("st.release.gpu.global.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
__device__ __forceinline__ unsigned int ld_relaxed_gpu(const unsigned int* p) {
  unsigned int v;
  asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(v) : "l"(p) : "memory");
  return v;
}

template <int OP, int TY>
__global__ void __launch_bounds__(NT, 1) k6_resident(const __grid_constant__ StencilParams p,
                                                     const __grid_constant__ CUtensorMap tmap,
                                                     const __grid_constant__ CUtensorMap pwmap, float* s0, float* s1,
                                                     int n_steps, int ntx, int nty) {
  constexpr bool PW = OP == K2C_HOTSPOT;
  constexpr int BY = TY + 2;
  constexpr int PLF = BY * BX;               // floats per box plane
  extern __shared__ __align__(128) float dsm[];
  __shared__ uint64_t bar;
  __shared__ int slot_sm;
  Geo G;
  G.nz = (int)p.n[0];
  G.ny = (int)p.n[1];
  G.nx = (int)p.n[2];
  const int tx = blockIdx.x % ntx, tyi = blockIdx.x / ntx;
  G.x0 = tx * TX;
  G.y0 = tyi * TY;
  G.hv = min(TY, G.ny - G.y0);
  G.wv = min(TX, G.nx - G.x0);
  const int boxf = ((PLF * G.nz + 31) / 32) * 32;      // floats per box, 128-B multiple
  float* const box0 = dsm;
  float* const box1 = dsm + boxf;
  float* pb = dsm + 2 * boxf;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;

  if (threadIdx.x == 0) {
    mbar_init(&bar, 1);
    fence_mbar_init();
    slot_sm = claim_slot<kSlots>(g_k6);
  }
  __syncthreads();
  K6Slot& S = g_k6[slot_sm];
  if (threadIdx.x == 0) {
    const uint32_t bytes = (uint32_t)(PLF * G.nz * 4) + (PW ? (uint32_t)(TX * TY * G.nz * 4) : 0u);
    mbar_arrive_expect_tx(&bar, bytes);
    tma_load_3d(box0, &tmap, &bar, G.x0 - XH, G.y0 - 1, 0);
    if constexpr (PW) tma_load_3d(pb, &pwmap, &bar, G.x0, G.y0, 0);
  }
  // the tiles whose edge cells fill this tile's halo: the face neighbours
  // (wrapping around under WRAP; none across a non-periodic grid edge)
  int nb = -1;
  if (threadIdx.x < 4) {
    const int d = threadIdx.x;
    int ax = tx, ay = tyi;
    const bool wx = p.kind[2] == PAD_WRAP, wy = p.kind[1] == PAD_WRAP;
    if (d == 0) ax = tx > 0 ? tx - 1 : (wx ? ntx - 1 : -1);
    if (d == 1) ax = tx + 1 < ntx ? tx + 1 : (wx ? 0 : -1);
    if (d == 2) ay = tyi > 0 ? tyi - 1 : (wy ? nty - 1 : -1);
    if (d == 3) ay = tyi + 1 < nty ? tyi + 1 : (wy ? 0 : -1);
    if (ax >= 0 && ay >= 0) nb = ay * ntx + ax;
  }
  mbar_wait(&bar, 0);
  // step 0's halo from the input itself (TMA's out-of-grid zeros replaced by the pad)
  fill_halo<BY>(p, G, box0, s0, threadIdx.x);
  __syncthreads();

  const int kz = p.kind[0];
  const float pv = p.pad_value;
  const int xo = G.x0 + 4 * lane;
  const bool x_ok = 4 * lane < G.wv;
  const int nrows = G.nz * TY;
  for (int t = 0; t < n_steps; ++t) {
    const float* src = (t & 1) ? box1 : box0;
    float* dstb = (t & 1) ? box0 : box1;
    const bool last = t + 1 == n_steps;
    float* gout = (t & 1) ? s0 : s1;            // the state buffer of step t+1 (iterate's ping-pong)
    for (int r = warp; r < nrows; r += NW) {
      const int z = r / TY, yy = r - z * TY;
      const int zmi = z > 0 ? z - 1 : (kz == PAD_CONSTANT ? -1 : (int)pad_remap(-1, G.nz, kz));
      const int zpi = z + 1 < G.nz ? z + 1 : (kz == PAD_CONSTANT ? -1 : (int)pad_remap(G.nz, G.nz, kz));
      const int off = z * PLF + (yy + 1) * BX + XH + 4 * lane;
      ColWin w;
      colwin_load(w, src + off, BX, PLF, zmi - z, zpi - z, zmi < 0, zpi < 0, pv, lane);
      float4 pw = make_float4(0.f, 0.f, 0.f, 0.f);
      if constexpr (PW) pw = lds128(pb + (z * TY + yy) * TX + 4 * lane);
      float4 res;
      res.x = colwin_eval<OP, 0>(p, w, pw);
      res.y = colwin_eval<OP, 1>(p, w, pw);
      res.z = colwin_eval<OP, 2>(p, w, pw);
      res.w = colwin_eval<OP, 3>(p, w, pw);
      *reinterpret_cast<float4*>(dstb + off) = res;
      if (last && x_ok && yy < G.hv) stg128(gout + ((int64_t)z * G.ny + G.y0 + yy) * G.nx + xo, res);
    }
    if (last) break;
    __syncthreads();
    store_edges<BY>(G, dstb, gout, threadIdx.x);
    // point-to-point step flags instead of a grid barrier: publish this
    // tile's edges of step t+1, wait for the (<= 4) tiles whose edges fill
    // the halo.  A tile overwrites a buffer's edges two steps later only
    // after its neighbours raised the flag of the step in between, i.e.
    // after they finished reading them.
    __syncthreads();
    if (threadIdx.x == 0) {
      __threadfence();
      st_release_gpu(&S.flag[blockIdx.x], (unsigned)(t + 1));
    }
    if (nb >= 0) {
      while ((int)(ld_relaxed_gpu(&S.flag[nb]) - (unsigned)(t + 1)) < 0) __nanosleep(20);
      asm volatile("fence.acq_rel.gpu;" ::: "memory");
    }
    __syncthreads();
    fill_halo<BY>(p, G, dstb, gout, threadIdx.x);
    __syncthreads();
  }
  // the last CTA out zeroes the flags and frees the slot
  if (threadIdx.x == 0 && atomicAdd(&S.exits, 1u) == gridDim.x - 1) {
    for (int i = 0; i < (int)gridDim.x; ++i) S.flag[i] = 0u;
    S.exits = 0u;
    __threadfence();
    atomicExch(&S.owner, 0ull);
  }
}

struct Launcher {
  const void* fn;
  size_t max_dyn;     // dynamic shared memory available next to the kernel's static shared memory
};

template <int OP, int TY>
Launcher get_launcher() {
  static Launcher L{};
  static std::once_flag once;
  std::call_once(once, [] {
    auto fn = k6_resident<OP, TY>;
    int dev = 0, optin = 0;
    cudaGetDevice(&dev);
    cudaDeviceGetAttribute(&optin, cudaDevAttrMaxSharedMemoryPerBlockOptin, dev);
    cudaFuncAttributes fa{};
    cudaFuncGetAttributes(&fa, fn);
    const size_t max_dyn = optin > (int)fa.sharedSizeBytes ? (size_t)optin - fa.sharedSizeBytes : 0;
    cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)max_dyn);
    cudaGetLastError();
    L = Launcher{reinterpret_cast<const void*>(fn), max_dyn};
  });
  return L;
}

constexpr int kTY[] = {2, 4, 8, 14, 16, 24, 32};

template <int OP>
Launcher launcher_for(int ty) {
  switch (ty) {
    case 2: return get_launcher<OP, 2>();
    case 4: return get_launcher<OP, 4>();
    case 8: return get_launcher<OP, 8>();
    case 14: return get_launcher<OP, 14>();
    case 16: return get_launcher<OP, 16>();
    case 24: return get_launcher<OP, 24>();
    default: return get_launcher<OP, 32>();
  }
}

Launcher launcher_for(int op, int ty) {
  return op == OP_HOTSPOT3D ? launcher_for<K2C_HOTSPOT>(ty) : launcher_for<K2C_WSTAR>(ty);
}

size_t smem_bytes(int ty, int nz, bool pw) {
  const size_t boxf = ((size_t)(BX * (ty + 2) * nz + 31) / 32) * 32;
  return 2 * boxf * 4 + (pw ? (size_t)TX * ty * nz * 4 : 0);
}

// the smallest compiled tile height whose tiles all fit on the device at
// once (one CTA per SM): the most parallel layout; 0 if none fits
int choose_ty(const StencilParams& p, int num_sms) {
  const int ntx = (int)((p.n[2] + TX - 1) / TX);
  const bool pw = p.op == OP_HOTSPOT3D;
  for (int ty : kTY) {
    const int64_t tiles = (int64_t)ntx * ((p.n[1] + ty - 1) / ty);
    if (tiles > num_sms || tiles > kMaxTiles) continue;
    if (smem_bytes(ty, (int)p.n[0], pw) > launcher_for(p.op, ty).max_dyn) return 0;
    return ty;
  }
  return 0;
}

}  // namespace

// Iterated few-plane 3D radius-1 star grids that fit in the device's shared
// memory (one tile per SM).  LIFT_K6=0 disables it (A/B).
bool resident3d_supported(const StencilParams& p, const float* s0, const float* s1, const float* aux,
                          int num_sms) {
  // opt-in (LIFT_K6=1): measured slower than per-step K2C launches replayed
  // from a CUDA graph on Hotspot3D 8x512x512 x100 (8.4 vs 6.6 us per step,
  // DESIGN.md §4): the per-step flag hand-off between SMs costs more than a
  // PDL launch hand-off
  const char* e = getenv("LIFT_K6");
  if (!(e && e[0] == '1')) return false;
  if (p.slab || p.n[0] > kMaxNz || p.radius != 1 || has_dampen(p)) return false;
  if (p.op != OP_HOTSPOT3D && p.op != OP_WEIGHTED) return false;
  for (int d = 0; d < 3; ++d)
    if (p.size[d] != 3 || p.lo[d] != 1 || p.hi[d] != 1 || p.step[d] != 1) return false;
  if (p.op == OP_WEIGHTED) {
    for (int k = 0; k < 27; ++k) {
      const int kz = k / 9, ky = (k / 3) % 3, kxx = k % 3;
      if ((kz != 1) + (ky != 1) + (kxx != 1) > 1 && p.wbox[k] != 0.0f) return false;   // star only
    }
  }
  if (p.n[2] % 4 != 0) return false;
  auto al = [](const void* q) { return (reinterpret_cast<uintptr_t>(q) & 15u) == 0; };
  if (!al(s0) || !al(s1) || (aux && !al(aux))) return false;
  return choose_ty(p, num_sms) > 0;
}

cudaError_t launch_resident3d(const StencilParams& p, float* s0, float* s1, const float* aux, int n_steps,
                              cudaStream_t stream, int num_sms, std::string* err) {
  const int ty = choose_ty(p, num_sms);
  if (ty <= 0) {
    *err = "K6: grid does not fit in shared memory";
    return cudaErrorInvalidConfiguration;
  }
  const bool pw = p.op == OP_HOTSPOT3D;
  const Launcher L = launcher_for(p.op, ty);
  const int nz = (int)p.n[0];
  CUtensorMap map, pwmap;
  if (!encode_tensor_map_3d(&map, s0, p.n[2], p.n[1], nz, BX, (uint32_t)(ty + 2), (uint32_t)nz, err))
    return cudaErrorInvalidValue;
  if (pw) {
    if (!encode_tensor_map_3d(&pwmap, aux, p.n[2], p.n[1], nz, TX, (uint32_t)ty, (uint32_t)nz, err))
      return cudaErrorInvalidValue;
  } else {
    pwmap = map;
  }
  const int ntx = (int)((p.n[2] + TX - 1) / TX);
  const int nty = (int)((p.n[1] + ty - 1) / ty);
  const int grid = ntx * nty;
  int n = n_steps, ntx_i = ntx, nty_i = nty;
  void* args[] = {(void*)&p, (void*)&map, (void*)&pwmap, (void*)&s0, (void*)&s1, &n, &ntx_i, &nty_i};
  cudaLaunchConfig_t cfg{};
  cfg.gridDim = dim3((unsigned)grid);
  cfg.blockDim = dim3(NT);
  cfg.dynamicSmemBytes = smem_bytes(ty, nz, pw);
  cfg.stream = stream;
  cudaLaunchAttribute at[1];
  at[0].id = cudaLaunchAttributeCooperative;      // co-residency for the step flags (or the launch fails)
  at[0].val.cooperative = 1;
  cfg.attrs = at;
  cfg.numAttrs = 1;
  set_last_kernel("k6_resident");
  return cudaLaunchKernelExC(&cfg, L.fn, args);
}

}  // namespace lift
