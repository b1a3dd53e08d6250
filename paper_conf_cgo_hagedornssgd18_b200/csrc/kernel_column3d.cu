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

// ---------------------------------------------------------------------------
// K2CT: two time steps of a few-plane grid per launch (temporal blocking of
// the whole-column tile; Hotspot3D's 8 planes).  The slid grid's box carries
// two halo rows / columns ((128+8) x (TY+4) x nz at (x0-4, y0-2)), the
// point-wise grid's box one ((128+8) x (TY+2) x nz at (x0-4, y0-1)).  Phase 1
// computes X_{t+1} on the tile plus one row / column around it into
// registers (lanes: the 128 columns; 2 (TY+2) nz threads: the halo columns
// x0-1 and x0+128); after a barrier X_{t+1} overwrites the slid box (same
// layout, rows y0-1 .. y0+TY), its out-of-grid cells take the remapped cell's
// value (pad of X_{t+1}, CLAMP / MIRROR / REFLECT), and phase 2 computes
// X_{t+2} on the tile.  One load latency and one launch per two steps; every
// value goes through colwin_eval (the operation sequence of single steps).
// ---------------------------------------------------------------------------
template <int I>
struct PtAcc {                   // one point of a box: x taps +-1, y taps +-BX, z taps dzm / dzp planes
  const float* c;
  int bxf, plf, dzm, dzp;
  template <int DZ, int DY, int DX>
  __device__ __forceinline__ float at() const {
    if constexpr (DZ < 0) return c[dzm * plf];
    else if constexpr (DZ > 0) return c[dzp * plf];
    else if constexpr (DY != 0) return c[DY * bxf];
    else return c[DX];
  }
};

template <int OP>
__device__ __forceinline__ float pt_eval(const StencilParams& p, const float* c, int bxf, int plf, int dzm, int dzp,
                                         float pw) {
  PtAcc<0> a{c, bxf, plf, dzm, dzp};
  if constexpr (OP == K2C_WSTAR) return op_weighted<1, 1, 1, true>(a, p.wbox);
  else return op_hotspot3d(a, pw, p.prm);
}

// remapped plane offsets of plane z's taps (reindexing kinds: inside [0, nz))
__device__ __forceinline__ void zoffs(int z, int nz, int kz, int& dzm, int& dzp) {
  const int zm = z > 0 ? z - 1 : (int)pad_remap(-1, nz, kz);
  const int zp = z + 1 < nz ? z + 1 : (int)pad_remap(nz, nz, kz);
  dzm = zm - z;
  dzp = zp - z;
}

template <int OP, int TY, int NZMAX>
__global__ void __launch_bounds__(NT, NZMAX <= 8 ? 3 : 1) k2ct_column(const __grid_constant__ StencilParams p,
                                                  const __grid_constant__ CUtensorMap tmap,
                                                  const __grid_constant__ CUtensorMap pwmap, float* __restrict__ out,
                                                  int ntx) {
  constexpr bool PW = OP == K2C_HOTSPOT;
  constexpr int BY = TY + 4;       // slid box rows y0-2 .. y0+TY+1
  constexpr int BY1 = TY + 2;      // X_{t+1} / point-wise rows y0-1 .. y0+TY
  constexpr int R1 = (BY1 * NZMAX + NW - 1) / NW;     // phase-1 rows per warp (upper bound)
  extern __shared__ __align__(128) float dsm[];
  __shared__ uint64_t bar;
  const int nz = (int)p.n[0], ny = (int)p.n[1], nx = (int)p.n[2];
  const int kx = p.kind[2], ky = p.kind[1], kz = p.kind[0];
  const int tbytes = BX * BY * nz * 4;
  const int tfl = ((tbytes + 127) / 128) * 32;
  float* tb = dsm;                 // slid box, then X_{t+1}
  float* pb = dsm + tfl;           // point-wise box
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int x0 = (blockIdx.x % ntx) * TX, y0 = (blockIdx.x / ntx) * TY;
  const int plf = BY * BX, plf1 = BY1 * BX;

  if (threadIdx.x == 0) {
    mbar_init(&bar, 1);
    fence_mbar_init();
  }
  __syncthreads();
  pdl_launch_dependents();
  pdl_wait();
  if (threadIdx.x == 0) {
    const uint32_t bytes = (uint32_t)tbytes + (PW ? (uint32_t)(BX * BY1 * nz * 4) : 0u);
    mbar_arrive_expect_tx(&bar, bytes);
    tma_load_3d(tb, &tmap, &bar, x0 - XH, y0 - 2, 0);
    if constexpr (PW) tma_load_3d(pb, &pwmap, &bar, x0 - XH, y0 - 1, 0);
  }
  mbar_wait(&bar, 0);

  // ---- pad of X_t: out-of-grid cells of the slid box <- the remapped cell ----
  // Only the cells a later read uses: box columns 2 .. TX+5 (x0-2 .. x0+129),
  // the out-of-grid rows among y0-2, y0-1 / ny, ny+1 (whole width) and the
  // out-of-grid columns among x0-2, x0-1 / nx, nx+1 (in-grid rows).  Every
  // source has both coordinates remapped into the grid, so it is never a
  // rewritten cell and the order of the writes does not matter.
  const bool x_edge = x0 == 0 || x0 + TX + 2 > nx;
  const bool y_edge = y0 == 0 || y0 + TY + 2 > ny;
  if (x_edge || y_edge) {
    const int rb = ny - (y0 - 2);                       // box row of gy = ny
    const int cb = nx - (x0 - XH);                      // box column of gx = nx
    const int nrt = y0 == 0 ? 2 : 0, nrb = rb < BY ? min(2, BY - rb) : 0;
    const int ncl = x0 == 0 ? 2 : 0, ncr = cb <= TX + XH + 1 ? min(2, TX + XH + 2 - cb) : 0;
    constexpr int W = TX + 4;                           // columns 2 .. TX+5
    const int nrow = nrt + nrb, ncol = ncl + ncr;
    const int per = nrow * W + ncol * BY;
    for (int c = threadIdx.x; c < nz * per; c += NT) {
      const int z = c / per, q = c - z * per;
      int r, col;
      if (q < nrow * W) {
        const int k = q / W;
        col = 2 + (q - k * W);
        r = k < nrt ? k : rb + (k - nrt);
      } else {
        const int q2 = q - nrow * W, k = q2 / BY;
        r = q2 - k * BY;
        col = k < ncl ? 2 + k : cb + (k - ncl);
        const int gyr = y0 - 2 + r;
        if (gyr < 0 || gyr >= ny) continue;              // (done by the row part)
      }
      int gy = y0 - 2 + r, gx = x0 - XH + col;
      if (gy < 0 || gy >= ny) gy = (int)pad_remap(gy, ny, ky);
      if (gx < 0 || gx >= nx) gx = (int)pad_remap(gx, nx, kx);
      const int br = gy - (y0 - 2), bc = gx - (x0 - XH);
      if (br >= 0 && br < BY && bc >= 0 && bc < BX) tb[z * plf + r * BX + col] = tb[z * plf + br * BX + bc];
    }
    __syncthreads();
  }

  // ---- phase 1: X_{t+1} on rows y0-1 .. y0+TY into registers ----
  const int xo = x0 + 4 * lane;
  const int nrows1 = nz * BY1;
  float4 x1[R1];
#pragma unroll
  for (int k = 0; k < R1; ++k) {
    const int r = warp + k * NW;
    if (r < nrows1) {
      const int z = r / BY1, r1 = r - z * BY1;       // X_{t+1} row r1 <-> box row r1 + 1
      int dzm, dzp;
      zoffs(z, nz, kz, dzm, dzp);
      const float* pl = tb + z * plf + (r1 + 1) * BX + XH + 4 * lane;
      ColWin w;
      colwin_load(w, pl, BX, plf, dzm, dzp, false, false, 0.0f, lane);
      float4 pw = make_float4(0.f, 0.f, 0.f, 0.f);
      if constexpr (PW) pw = lds128(pb + (z * BY1 + r1) * BX + XH + 4 * lane);
      x1[k].x = colwin_eval<OP, 0>(p, w, pw);
      x1[k].y = colwin_eval<OP, 1>(p, w, pw);
      x1[k].z = colwin_eval<OP, 2>(p, w, pw);
      x1[k].w = colwin_eval<OP, 3>(p, w, pw);
    }
  }
  // halo columns x0-1 / x0+128 of X_{t+1}: one point per thread
  float xh = 0.0f;
  const int nh = 2 * nrows1;
  int hidx = -1;
  if ((int)threadIdx.x < nh) {
    const int side = threadIdx.x / nrows1, r = threadIdx.x - side * nrows1;
    const int z = r / BY1, r1 = r - z * BY1;
    const int col = side ? XH + TX : XH - 1;
    int dzm, dzp;
    zoffs(z, nz, kz, dzm, dzp);
    const float* c = tb + z * plf + (r1 + 1) * BX + col;
    const float pw = PW ? pb[(z * BY1 + r1) * BX + col] : 0.0f;
    xh = pt_eval<OP>(p, c, BX, plf, dzm, dzp, pw);
    hidx = z * plf1 + r1 * BX + col;
  }
  __syncthreads();               // every read of X_t is done
  // X_{t+1} box (same memory): plane z, row r1 <-> y0-1+r1, column XH+i <-> x0+i
#pragma unroll
  for (int k = 0; k < R1; ++k) {
    const int r = warp + k * NW;
    if (r < nrows1) {
      const int z = r / BY1, r1 = r - z * BY1;
      *reinterpret_cast<float4*>(tb + z * plf1 + r1 * BX + XH + 4 * lane) = x1[k];
    }
  }
  if (hidx >= 0) tb[hidx] = xh;
  __syncthreads();
  // pad of X_{t+1}: the out-of-grid row / column next to the grid (y0-1 = -1 /
  // ny; x0-1 = -1 / nx) <- its remapped in-grid row / column
  if (x_edge || y_edge) {
    const int rb = ny - (y0 - 1);                       // X_{t+1} row of gy = ny
    const int cb = nx - (x0 - XH);                      // column of gx = nx
    const int nrt = y0 == 0 ? 1 : 0, nrb = rb < BY1 ? 1 : 0;
    const int ncl = x0 == 0 ? 1 : 0, ncr = cb <= TX + XH ? 1 : 0;
    constexpr int W = TX + 2;                           // columns XH-1 .. XH+TX
    const int nrow = nrt + nrb, ncol = ncl + ncr;
    const int per = nrow * W + ncol * BY1;
    for (int c = threadIdx.x; c < nz * per; c += NT) {
      const int z = c / per, q = c - z * per;
      int r1, col;
      if (q < nrow * W) {
        const int k = q / W;
        col = XH - 1 + (q - k * W);
        r1 = k < nrt ? 0 : rb;
      } else {
        const int q2 = q - nrow * W, k = q2 / BY1;
        r1 = q2 - k * BY1;
        col = k < ncl ? XH - 1 : cb;
        const int gyr = y0 - 1 + r1;
        if (gyr < 0 || gyr >= ny) continue;              // (done by the row part)
      }
      int gy = y0 - 1 + r1, gx = x0 - XH + col;
      if (gy < 0 || gy >= ny) gy = (int)pad_remap(gy, ny, ky);
      if (gx < 0 || gx >= nx) gx = (int)pad_remap(gx, nx, kx);
      const int br = gy - (y0 - 1), bc = gx - (x0 - XH);
      if (br >= 0 && br < BY1 && bc >= XH - 1 && bc <= XH + TX)
        tb[z * plf1 + r1 * BX + col] = tb[z * plf1 + br * BX + bc];
    }
    __syncthreads();
  }
  // ---- phase 2: X_{t+2} on the tile ----
  const bool x_ok = xo < nx;
  const int nrows2 = nz * TY;
  for (int r = warp; r < nrows2; r += NW) {
    const int z = r / TY, yy = r - z * TY;
    const int gy = y0 + yy;
    int dzm, dzp;
    zoffs(z, nz, kz, dzm, dzp);
    const float* pl = tb + z * plf1 + (yy + 1) * BX + XH + 4 * lane;
    ColWin w;
    colwin_load(w, pl, BX, plf1, dzm, dzp, false, false, 0.0f, lane);
    float4 pw = make_float4(0.f, 0.f, 0.f, 0.f);
    if constexpr (PW) pw = lds128(pb + (z * BY1 + yy + 1) * BX + XH + 4 * lane);
    float4 res;
    res.x = colwin_eval<OP, 0>(p, w, pw);
    res.y = colwin_eval<OP, 1>(p, w, pw);
    res.z = colwin_eval<OP, 2>(p, w, pw);
    res.w = colwin_eval<OP, 3>(p, w, pw);
    if (x_ok && gy < ny) stg128(out + ((int64_t)z * ny + gy) * nx + xo, res);
  }
}

template <int OP, int TY, int NZMAX>
Launcher get_launcher_t2() {
  static Launcher L{};
  static std::once_flag once;
  std::call_once(once, [] {
    auto fn = k2ct_column<OP, TY, NZMAX>;
    const int max_smem = ((BX * (TY + 4) * kMaxNz * 4 + 127) / 128) * 128 + BX * (TY + 2) * kMaxNz * 4;
    cudaFuncSetAttribute(fn, cudaFuncAttributeMaxDynamicSharedMemorySize, max_smem);
    cudaGetLastError();
    L = Launcher{reinterpret_cast<const void*>(fn), TY};
  });
  return L;
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

namespace lift {

// Two steps per launch (K2CT) for the plans K2C takes, with reindexing pads
// only (the out-of-grid X_{t+1} cells are copies of in-grid ones); not
// slabbed; LIFT_K2CT=0 disables.
bool column3d_t2_supported(const StencilParams& p, const float* in0, const float* in1) {
  const char* e = getenv("LIFT_K2CT");
  if (e && e[0] == '0') return false;
  if (!sweep3d_supported(p) || !column3d_supported(p, in0, in1)) return false;
  if (p.op != OP_HOTSPOT3D) return false;
  for (int d = 0; d < 3; ++d)
    if (p.kind[d] != PAD_CLAMP && p.kind[d] != PAD_MIRROR && p.kind[d] != PAD_REFLECT) return false;
  return true;
}

cudaError_t launch_column3d_t2(const StencilParams& p, const float* in0, const float* in1, float* out,
                               cudaStream_t stream, std::string* err) {
  const char* e = getenv("LIFT_K2CT_TY");
  const int ty = e ? atoi(e) : 5;
  const int nz = (int)p.n[0];
  Launcher L;
  if (nz <= 8)
    L = ty == 4 ? get_launcher_t2<K2C_HOTSPOT, 4, 8>() : get_launcher_t2<K2C_HOTSPOT, 5, 8>();
  else
    L = ty == 4 ? get_launcher_t2<K2C_HOTSPOT, 4, kMaxNz>() : get_launcher_t2<K2C_HOTSPOT, 5, kMaxNz>();
  CUtensorMap map, pwmap;
  if (!get_map(in0, p.n[2], p.n[1], nz, BX, L.ty + 4, &map, err)) return cudaErrorInvalidValue;
  if (!get_map(in1, p.n[2], p.n[1], nz, BX, L.ty + 2, &pwmap, err)) return cudaErrorInvalidValue;
  const int ntx = (int)((p.n[2] + TX - 1) / TX);
  const int64_t nty = (p.n[1] + L.ty - 1) / L.ty;
  const int64_t grid = ntx * nty;
  if (grid > 0x7fffffff) return cudaErrorInvalidConfiguration;
  const size_t smem = ((BX * (L.ty + 4) * nz * 4 + 127) / 128) * 128 + (size_t)BX * (L.ty + 2) * nz * 4;
  int ntx_i = ntx;
  void* args[] = {(void*)&p, (void*)&map, (void*)&pwmap, (void*)&out, &ntx_i};
  set_last_kernel("k2ct_column");
  return launch_kernel(L.fn, dim3((unsigned)grid), dim3(NT), args, smem, stream, true);
}

}  // namespace lift
