/* c_abi_demo.c — drive libstencil.so through include/stencil.h from plain C
 * (no Python, no torch): J3D7 on a seeded grid, 3 iterated steps with
 * stencil_run_host (host buffers in/out), then one stencil_apply on device
 * buffers.  Writes the two results as raw float32 to argv[1] / argv[2]
 * (tests/test_c_abi_gpu.py checks them against the fp64 oracle).
 *
 *   gcc -O2 -std=c99 -I include examples/c_abi_demo.c \
 *       -L paper_conf_cgo_hagedornssgd18_b200 -lstencil -lcudart -o c_abi_demo
 */
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>

#include "stencil.h"

/* device memory through the CUDA runtime, declared here to keep the demo
 * free of CUDA headers */
extern int cudaMalloc(void** p, size_t n);
extern int cudaMemcpy(void* d, const void* s, size_t n, int kind);
extern int cudaFree(void* p);
extern int cudaDeviceSynchronize(void);

#define CHECK(x)                                                                        \
  do {                                                                                  \
    stencil_status s_ = (x);                                                            \
    if (s_ != STENCIL_OK) {                                                             \
      fprintf(stderr, "%s failed: %s (%s)\n", #x, stencil_status_string(s_), stencil_last_error()); \
      return 1;                                                                         \
    }                                                                                   \
  } while (0)

int main(int argc, char** argv) {
  if (argc < 3) {
    fprintf(stderr, "usage: %s out_iterate.f32 out_apply.f32\n", argv[0]);
    return 2;
  }
  const int64_t ext[3] = {20, 36, 132};
  const int32_t size[3] = {3, 3, 3}, step[3] = {1, 1, 1}, lo[3] = {1, 1, 1}, hi[3] = {1, 1, 1};
  const int32_t kind[3] = {STENCIL_PAD_CLAMP, STENCIL_PAD_MIRROR, STENCIL_PAD_WRAP};
  float w[27] = {0};
  w[13] = 0.40f; w[4] = 0.05f; w[22] = 0.15f; w[10] = 0.10f; w[16] = 0.10f; w[12] = 0.08f; w[14] = 0.12f;
  const size_t n = (size_t)(ext[0] * ext[1] * ext[2]);
  float* x = malloc(n * sizeof(float));
  float* y = malloc(n * sizeof(float));
  uint32_t st = 12345u;
  for (size_t i = 0; i < n; ++i) {          /* LCG, values in [0.5, 1.5) */
    st = st * 1664525u + 1013904223u;
    x[i] = 0.5f + (float)(st >> 8) / 16777216.0f;
  }
  FILE* fx = fopen("c_abi_demo_input.f32", "wb");
  fwrite(x, sizeof(float), n, fx);
  fclose(fx);

  stencil_plan plan;
  CHECK(stencil_plan_create(&plan, 0, 3, ext, size, step, lo, hi, kind, 0.0f, STENCIL_OP_WEIGHTED, w, NULL, 0));
  printf("%s, variant %d\n", stencil_version(), stencil_plan_variant(plan));

  const float* hs[1] = {x};
  CHECK(stencil_run_host(plan, hs, 1, NULL, 0, 3, y, NULL));
  FILE* f1 = fopen(argv[1], "wb");
  fwrite(y, sizeof(float), n, f1);
  fclose(f1);

  void *dx = NULL, *dy = NULL;
  if (cudaMalloc(&dx, n * sizeof(float)) || cudaMalloc(&dy, n * sizeof(float))) return 3;
  cudaMemcpy(dx, x, n * sizeof(float), 1 /* H2D */);
  const float* in[1] = {(const float*)dx};
  CHECK(stencil_apply(plan, in, 1, (float*)dy, NULL));
  if (cudaDeviceSynchronize()) return 4;
  cudaMemcpy(y, dy, n * sizeof(float), 2 /* D2H */);
  FILE* f2 = fopen(argv[2], "wb");
  fwrite(y, sizeof(float), n, f2);
  fclose(f2);

  /* error behaviour: out aliasing the slid input is rejected synchronously */
  if (stencil_apply(plan, in, 1, (float*)dx, NULL) != STENCIL_E_INVALID) return 5;
  cudaFree(dx);
  cudaFree(dy);
  stencil_plan_destroy(plan);
  free(x);
  free(y);
  printf("ok\n");
  return 0;
}
