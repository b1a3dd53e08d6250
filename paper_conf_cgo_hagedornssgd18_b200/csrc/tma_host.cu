// tma_host.cu — cuTensorMapEncodeTiled through the runtime's driver entry
// point (the library links the static CUDA runtime only, never -lcuda).
#include <cuda.h>
#include <cuda_runtime.h>

#include <cstdlib>
#include <mutex>
#include <string>

#include "launch.hpp"

namespace lift {
namespace {

typedef CUresult (*EncodeTiledFn)(CUtensorMap*, CUtensorMapDataType, cuuint32_t, void*, const cuuint64_t*,
                                  const cuuint64_t*, const cuuint32_t*, const cuuint32_t*, CUtensorMapInterleave,
                                  CUtensorMapSwizzle, CUtensorMapL2promotion, CUtensorMapFloatOOBfill);

EncodeTiledFn get_encoder(std::string* err) {
  static EncodeTiledFn fn = nullptr;
  static std::once_flag once;
  static std::string init_err;
  std::call_once(once, [] {
    void* p = nullptr;
    cudaDriverEntryPointQueryResult q;
    cudaError_t e = cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q);
    if (e != cudaSuccess || q != cudaDriverEntryPointSuccess || !p) {
      init_err = "cuTensorMapEncodeTiled entry point unavailable";
      cudaGetLastError();
      return;
    }
    fn = reinterpret_cast<EncodeTiledFn>(p);
  });
  if (!fn && err) *err = init_err;
  return fn;
}

}  // namespace

bool encode_tensor_map_3d(CUtensorMap* map, const float* base, int64_t nx, int64_t ny, int64_t nz,
                          uint32_t box_x, uint32_t box_y, uint32_t box_z, std::string* err) {
  EncodeTiledFn fn = get_encoder(err);
  if (!fn) return false;
  const cuuint64_t dims[3] = {(cuuint64_t)nx, (cuuint64_t)ny, (cuuint64_t)nz};
  const cuuint64_t strides[2] = {(cuuint64_t)nx * sizeof(float), (cuuint64_t)nx * ny * sizeof(float)};
  const cuuint32_t box[3] = {box_x, box_y, box_z};
  const cuuint32_t estr[3] = {1, 1, 1};
  // L2 promotion (tuning hook LIFT_L2PROMO = 0 none, 1 64B, 2 128B, 3 256B)
  static const int promo = [] { const char* e = getenv("LIFT_L2PROMO"); return e ? atoi(e) : 3; }();
  const CUtensorMapL2promotion pr = promo == 0 ? CU_TENSOR_MAP_L2_PROMOTION_NONE
                                    : promo == 1 ? CU_TENSOR_MAP_L2_PROMOTION_L2_64B
                                    : promo == 2 ? CU_TENSOR_MAP_L2_PROMOTION_L2_128B
                                                 : CU_TENSOR_MAP_L2_PROMOTION_L2_256B;
  CUresult r = fn(map, CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 3, const_cast<float*>(base), dims, strides, box, estr,
                  CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE, pr, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  if (r != CUDA_SUCCESS) {
    if (err) *err = "cuTensorMapEncodeTiled failed (code " + std::to_string((int)r) + ")";
    return false;
  }
  return true;
}

}  // namespace lift
