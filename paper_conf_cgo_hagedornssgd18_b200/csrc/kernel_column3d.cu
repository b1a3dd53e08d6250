// kernel_column3d.cu — K2C: whole-column tiles for 3D grids with few planes.
//
// slide_3 over grids whose slowest extent is small (Hotspot3D's
// 8 planes, Table 1): the z-sweep of K2 streams each (z-chunk, tile)
// item plane by plane through a TMA ring, so on an 8-plane grid every CTA
// pays two or three serial load latencies for a handful of planes and the
// launch is latency-bound (ncu: 22% warps active, long-scoreboard stalls,
// 0.25 of HBM cold).  Here a CTA owns one 128 x TY (x, y) tile over ALL nz
// planes and issues its whole input in two TMA box loads at once (the slid
// grid (128+8) x (TY+2) x nz, the point-wise grid 128 x TY x nz): one load
// latency per CTA, every byte of the grid in flight from the first
// microsecond, no ticket counter, no producer warp.  The z taps of the edge
// planes are read from the remapped plane inside the box (pad h on z,
// every reindexing kind maps into [0, nz)); x/y pads are applied
// by rewriting the box's out-of-grid cells (halo.cuh) on edge tiles; the
// value pad in z is a register constant.  The map f is ops.cuh's, with the
// same operation sequence as every other kernel family (A12).
#include <cuda.h>
#include <cuda_runtime.h>

#include <cstdint>
#include <mutex>
#include <string>

#include "common.cuh"
#include "launch.hpp"
#include "ops.cuh"
#include "tma.cuh"
#include "colwin.cuh"

namespace lift {
namespace {

constexpr int TX = 128;
constexpr int XH = 4;
constexpr int BX = TX + 2 * XH;
constexpr int NW = 8;
constexpr int NT = NW * 32;
constexpr int kMaxNz = 16;

template <int OP, int TY>
__global__ void __launch_bounds__(NT) k2c_column(const __grid_constant__ StencilParams p,
                                                 const __grid_constant__ CUtensorMap tmap,
                                                 const __grid_constant__ CUtensorMap pwmap,
                                                 const float* __restrict__ src, float* __restrict__ out, int ntx) {
  constexpr bool PW = OP == K2C_HOTSPOT;
  constexpr int BY = TY + 2;
  extern __shared__ __align__(128) float dsm[];
  __shared__ uint64_t bar;
  const int nz = (int)p.n[0], ny = (int)p.n[1], nx = (int)p.n[2];
  const int tbytes = BX * BY * nz * 4;
  const int tfl = ((tbytes + 127) / 128) * 32;             // slid box floats, 128-B aligned
  float* tb = dsm;
  float* pb = dsm + tfl;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int x0 = (blockIdx.x % ntx) * TX, y0 = (blockIdx.x / ntx) * TY;

  if (threadIdx.x == 0) {
    mbar_init(&bar, 1);
    fence_mbar_init();
  }
  __syncthreads();
  pdl_launch_dependents();
  pdl_wait();
  if (threadIdx.x == 0) {
    const uint32_t bytes = (uint32_t)tbytes + (PW ? (uint32_t)(TX * TY * nz * 4) : 0u);
    mbar_arrive_expect_tx(&bar, bytes);
    tma_load_3d(tb, &tmap, &bar, x0 - XH, y0 - 1, 0);
    if constexpr (PW) tma_load_3d(pb, &pwmap, &bar, x0, y0, 0);
  }
  mbar_wait(&bar, 0);

  const int kx = p.kind[2], ky = p.kind[1], kz = p.kind[0];
  const float pv = p.pad_value;
  const bool x_edge = (x0 == 0) || (x0 + TX + 1 > nx);
  const bool y_edge = (y0 == 0) || (y0 + TY + 1 > ny);
  // TMA fills out-of-grid cells with zeros: right for a zero value pad,
  // rewritten here for the reindexing kinds and a non-zero constant
  const bool zero_pad = kx == PAD_CONSTANT && ky == PAD_CONSTANT && pv == 0.0f;
  if ((x_edge || y_edge) && !zero_pad) {
    // one flat loop over (plane, halo cell): a cell outside the grid gets the
    // constant, or input[h_y(gy), h_x(gx)] — read from the box when the
    // remapped cell lies in it (clamp / mirror / reflect: always), else from
    // global memory (wrap).  Sources are in-grid cells, which are never
    // rewritten, so the order of the writes does not matter.
    const int ncl = x0 == 0 ? 1 : 0;
    const int rc0 = nx - x0 + XH;                       // box column of gx = nx
    const int ncr = rc0 < BX ? 1 : 0;
    const int nrt = y0 == 0 ? 1 : 0;
    const int rr0 = ny - y0 + 1;                        // box row of gy = ny
    const int nrb = rr0 < BY ? 1 : 0;
    const int ccols = (ncl + ncr) * BY;
    const int per = ccols + (nrt + nrb) * BX;
    for (int c = threadIdx.x; c < nz * per; c += NT) {
      const int z = c / per, q = c - z * per;
      int r, col;
      if (q < ccols) {
        const int k = q / BY;
        r = q - k * BY;
        col = (k < ncl) ? XH - 1 : rc0;
      } else {
        const int k = (q - ccols) / BX;
        col = (q - ccols) - k * BX;
        r = (k < nrt) ? 0 : rr0;
      }
      int gy = y0 - 1 + r, gx = x0 - XH + col;
      const bool oy = gy < 0 || gy >= ny, ox = gx < 0 || gx >= nx;
      float v;
      if ((oy && ky == PAD_CONSTANT) || (ox && kx == PAD_CONSTANT)) {
        v = pv;
      } else {
        if (oy) gy = (int)pad_remap(gy, ny, ky);
        if (ox) gx = (int)pad_remap(gx, nx, kx);
        const int br = gy - (y0 - 1), bc = gx - (x0 - XH);
        v = (br >= 0 && br < BY && bc >= 0 && bc < BX) ? tb[(z * BY + br) * BX + bc]
                                                         : __ldg(src + ((int64_t)z * ny + gy) * nx + gx);
      }
      tb[(z * BY + r) * BX + col] = v;
    }
    __syncthreads();
  }

  const int xo = x0 + 4 * lane;
  const bool x_ok = xo < nx;
  const int nrows = nz * TY;
  for (int r = warp; r < nrows; r += NW) {
    const int z = r / TY, yy = r - z * TY;
    const int gy = y0 + yy;
    // z taps: the remapped plane (inside the box) or the value pad
    const int zmi = z > 0 ? z - 1 : (kz == PAD_CONSTANT ? -1 : (int)pad_remap(-1, nz, kz));
    const int zpi = z + 1 < nz ? z + 1 : (kz == PAD_CONSTANT ? -1 : (int)pad_remap(nz, nz, kz));
    const float* pl = tb + z * BY * BX + (yy + 1) * BX + XH + 4 * lane;
    ColWin w;
    colwin_load(w, pl, BX, BY * BX, zmi - z, zpi - z, zmi < 0, zpi < 0, pv, lane);
    float4 pw = make_float4(0.f, 0.f, 0.f, 0.f);
    if constexpr (PW) pw = lds128(pb + (z * TY + yy) * TX + 4 * lane);
    float4 res;
    res.x = colwin_eval<OP, 0>(p, w, pw);
    res.y = colwin_eval<OP, 1>(p, w, pw);
    res.z = colwin_eval<OP, 2>(p, w, pw);
    res.w = colwin_eval<OP, 3>(p, w, pw);
    if (x_ok && gy < ny) stg128(out + ((int64_t)z * ny + gy) * nx + xo, res);
  }
}

struct Launcher {
  const void* fn;
  int ty;
};

template <int OP, int TY>
Launcher get_launcher() {
  static Launcher L{};
  static std::once_flag once;
  std::call_once(once, [] {
    auto fn = k2c_column<OP, TY>;
    const int max_smem = ((BX * (TY + 2) * kMaxNz * 4 + 127) / 128) * 128 + TX * TY * kMaxNz * 4;
    cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, max_smem);
    cudaGetLastError();
    L = Launcher{reinterpret_cast<const void*>(fn), TY};
  });
  return L;
}

struct MapEntry {
  const float* base;
  int64_t nx, ny, nz;
  int bx, by;
  CUtensorMap map;
};

bool get_map(const float* base, int64_t nx, int64_t ny, int64_t nz, int bx, int by, CUtensorMap* out,
             std::string* err) {
  thread_local MapEntry cache[8];
  thread_local int next = 0;
  for (auto& e : cache)
    if (e.base == base && e.nx == nx && e.ny == ny && e.nz == nz && e.bx == bx && e.by == by) {
      *out = e.map;
      return true;
    }
  MapEntry e{base, nx, ny, nz, bx, by, {}};
  if (!encode_tensor_map_3d(&e.map, base, nx, ny, nz, (uint32_t)bx, (uint32_t)by, (uint32_t)nz, err)) return false;
  cache[next] = e;
  next = (next + 1) % 8;
  *out = e.map;
  return true;
}

int column_ty() {
  const char* e = getenv("LIFT_K2C_TY");      // A/B: tile rows
  return e ? atoi(e) : 4;
}

}  // namespace

// Few-plane 3D grids (nz <= 16) of the radius-1 star ops, whole region, not
// slabbed; the caller (launch_sweep3d) has already checked sweep3d_supported.
// LIFT_K2C=0 disables (A/B), LIFT_K2C=1 forces it for every eligible plan.
bool column3d_supported(const StencilParams& p, const float* in0, const float* in1) {
  const char* e = getenv("LIFT_K2C");
  if (e && e[0] == '0') return false;
  if (p.slab || p.reg0 != 0 || p.reg1 != p.n[0]) return false;
  if (p.put_lo || p.put_hi || p.fused_step || p.wait_lo || p.wait_hi) return false;
  if (p.radius != 1 || p.n[0] > kMaxNz) return false;
  if (p.op != OP_HOTSPOT3D && p.op != OP_WEIGHTED) return false;
  if (p.op == OP_WEIGHTED) {
    for (int k = 0; k < 27; ++k) {
      const int kz = k / 9, ky = (k / 3) % 3, kxx = k % 3;
      if ((kz != 1) + (ky != 1) + (kxx != 1) > 1 && p.wbox[k] != 0.0f) return false;   // star only
    }
  }
  if (p.n[2] % 4 != 0) return false;
  if ((reinterpret_cast<uintptr_t>(in0) & 15u) || (in1 && (reinterpret_cast<uintptr_t>(in1) & 15u))) return false;
  return true;
}

cudaError_t launch_column3d(const StencilParams& p, const float* in0, const float* in1, float* out,
                            cudaStream_t stream, std::string* err) {
  const int ty = column_ty();
  Launcher L;
  if (p.op == OP_HOTSPOT3D) L = ty == 8 ? get_launcher<K2C_HOTSPOT, 8>() : get_launcher<K2C_HOTSPOT, 4>();
  else L = ty == 8 ? get_launcher<K2C_WSTAR, 8>() : get_launcher<K2C_WSTAR, 4>();
  const int nz = (int)p.n[0];
  CUtensorMap map, pwmap;
  if (!get_map(in0, p.n[2], p.n[1], nz, BX, L.ty + 2, &map, err)) return cudaErrorInvalidValue;
  if (p.op == OP_HOTSPOT3D) {
    if (!get_map(in1, p.n[2], p.n[1], nz, TX, L.ty, &pwmap, err)) return cudaErrorInvalidValue;
  } else {
    pwmap = map;
  }
  const int ntx = (int)((p.n[2] + TX - 1) / TX);
  const int64_t nty = (p.n[1] + L.ty - 1) / L.ty;
  const int64_t grid = ntx * nty;
  if (grid > 0x7fffffff) return cudaErrorInvalidConfiguration;
  const size_t smem = ((BX * (L.ty + 2) * nz * 4 + 127) / 128) * 128 +
                      (p.op == OP_HOTSPOT3D ? (size_t)TX * L.ty * nz * 4 : 0);
  int ntx_i = ntx;
  void* args[] = {(void*)&p, (void*)&map, (void*)&pwmap, (void*)&in0, (void*)&out, &ntx_i};
  set_last_kernel("k2c_column");
  return launch_kernel(L.fn, dim3((unsigned)grid), dim3(NT), args, smem, stream, true);
}

}  // namespace lift
