// halo.cuh — boundary fix-up of a TMA-staged halo'd tile (edge tiles only).
//
// TMA fills cells outside the tensor with zeros.  For the reindexing pads
// (clamp / mirror / wrap / reflect) and for a non-zero constant
// the out-of-grid cells that the window can reach are rewritten
// here: cell (gy, gx) gets pad_value when an out-of-range dimension is
// CONSTANT, else input[h_y(gy), h_x(gx)] — the pad_n value for any order of
// the per-dimension pads (A9).  Interior tiles never run this.
#pragma once
#include "common.cuh"

namespace lift {

// Box layout: BX columns starting at x0 - XH, BY rows starting at y0 - RY.
// Only columns x in [-RX, 0) u [nx, nx + RX) and rows y in [-RY, 0) u
// [ny, ny + RY) that fall inside the box are rewritten.
template <int RY, int RX, int XH, int BX, int BY, int NTHREADS>
__device__ __forceinline__ void fixup_tile(const StencilParams& p, float* st, const float* __restrict__ src,
                                           int64_t lz, int x0, int y0, int tid) {
  const int64_t nx = p.n[2], ny = p.n[1];
  const int kx = p.kind[2], ky = p.kind[1];
  const int lcol0 = XH - RX;
  const int ncl = (x0 == 0) ? RX : 0;
  const int rc0 = (int)(nx - x0) + XH;
  const int ncr = (rc0 < BX) ? min(RX, BX - rc0) : 0;
  const int ncols = ncl + ncr;
  const int nrt = (y0 == 0) ? RY : 0;
  const int rr0 = (int)(ny - y0) + RY;
  const int nrb = (rr0 < BY) ? min(RY, BY - rr0) : 0;
  const int ncell_cols = ncols * BY;
  const int ncell = ncell_cols + (nrt + nrb) * BX;
  for (int c = tid; c < ncell; c += NTHREADS) {
    int r, col;
    if (c < ncell_cols) {
      const int k = c / BY;
      r = c % BY;
      col = (k < ncl) ? lcol0 + k : rc0 + (k - ncl);
    } else {
      const int k = (c - ncell_cols) / BX;
      col = (c - ncell_cols) % BX;
      r = (k < nrt) ? k : rr0 + (k - nrt);
    }
    int64_t gy = (int64_t)y0 - RY + r;
    int64_t gx = (int64_t)x0 - XH + col;
    const bool oy = gy < 0 || gy >= ny, ox = gx < 0 || gx >= nx;
    float v;
    if ((oy && ky == PAD_CONSTANT) || (ox && kx == PAD_CONSTANT)) {
      v = p.pad_value;
    } else {
      if (oy) gy = pad_remap(gy, ny, ky);
      if (ox) gx = pad_remap(gx, nx, kx);
      v = __ldg(src + lz * p.plane + gy * nx + gx);
    }
    st[r * BX + col] = v;
  }
}

}  // namespace lift
