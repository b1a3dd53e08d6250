// colwin.cuh — the radius-1 star window of one lane's 4 output columns in
// registers, shared by the whole-column kernels (K2C, K6): x taps from the
// lane's float4 and its neighbours, y/z taps from shared memory.  f is
// ops.cuh's (the operation sequence of every kernel family, A12).
#pragma once
#include "common.cuh"
#include "ops.cuh"
#include "tma.cuh"

namespace lift {

enum ColOp { K2C_WSTAR = 0, K2C_HOTSPOT = 1 };

struct ColWin {
  float x[6];     // centre row, x offsets -1 .. 4
  float ym[4], yp[4], zm[4], zp[4];
};

template <int I>
struct ColAcc {
  const ColWin& w;
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

__device__ __forceinline__ void colwin_set4(float (&d)[4], float4 v) {
  d[0] = v.x; d[1] = v.y; d[2] = v.z; d[3] = v.w;
}

template <int OP, int I>
__device__ __forceinline__ float colwin_eval(const StencilParams& p, const ColWin& w, const float4& pw) {
  ColAcc<I> a{w};
  if constexpr (OP == K2C_WSTAR) return op_weighted<1, 1, 1, true>(a, p.wbox);
  else return op_hotspot3d(a, f4get(pw, I), p.prm);
}

// The window of the lane's columns at box address ``pl`` (centre float4;
// rows BXF floats apart, planes PLF apart), z taps from planes zmi / zpi
// (-1: the value pad pv), x halo from the neighbour lanes / the box.
__device__ __forceinline__ void colwin_load(ColWin& w, const float* pl, int bxf, int plf, int dzm, int dzp, bool zm_c,
                                            bool zp_c, float pv, int lane) {
  const float4 c = lds128(pl);
  colwin_set4(w.ym, lds128(pl - bxf));
  colwin_set4(w.yp, lds128(pl + bxf));
  if (!zm_c) colwin_set4(w.zm, lds128(pl + dzm * plf));
  else w.zm[0] = w.zm[1] = w.zm[2] = w.zm[3] = pv;
  if (!zp_c) colwin_set4(w.zp, lds128(pl + dzp * plf));
  else w.zp[0] = w.zp[1] = w.zp[2] = w.zp[3] = pv;
  w.x[1] = c.x; w.x[2] = c.y; w.x[3] = c.z; w.x[4] = c.w;
  const float left = __shfl_up_sync(0xffffffffu, c.w, 1);
  const float right = __shfl_down_sync(0xffffffffu, c.x, 1);
  w.x[0] = lane == 0 ? pl[-1] : left;
  w.x[5] = lane == 31 ? pl[4] : right;
}

}  // namespace lift
