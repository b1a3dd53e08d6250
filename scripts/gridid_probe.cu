// gridid_probe.cu — checks that %gridid differs for every launch (eager, two
// streams, graph replays): the key of the per-launch counter slots (slots.cuh).
#include <cstdio>
#include <set>
#include <vector>
#include <cuda_runtime.h>
__global__ void k(unsigned long long* out, int i) {
  unsigned long long g;
  asm volatile("mov.u64 %0, %%gridid;" : "=l"(g));
  if (threadIdx.x == 0 && blockIdx.x == 0) out[i] = g;
}
int main() {
  const int N = 64;
  unsigned long long* d;
  cudaMalloc(&d, N * 8 * 4);
  cudaStream_t s1, s2;
  cudaStreamCreate(&s1);
  cudaStreamCreate(&s2);
  for (int i = 0; i < 8; ++i) k<<<2, 32, 0, (i & 1) ? s1 : s2>>>(d, i);
  cudaGraph_t g;
  cudaGraphExec_t ge;
  cudaStreamBeginCapture(s1, cudaStreamCaptureModeGlobal);
  for (int i = 0; i < 4; ++i) k<<<2, 32, 0, s1>>>(d, 8 + i);
  cudaStreamEndCapture(s1, &g);
  cudaGraphInstantiate(&ge, g, 0);
  std::vector<unsigned long long> all;
  std::vector<unsigned long long> h(N);
  cudaDeviceSynchronize();
  cudaMemcpy(h.data(), d, 8 * 8, cudaMemcpyDeviceToHost);
  for (int i = 0; i < 8; ++i) all.push_back(h[i]);
  for (int r = 0; r < 3; ++r) {
    cudaGraphLaunch(ge, r & 1 ? s1 : s2);
    cudaDeviceSynchronize();
    cudaMemcpy(h.data(), d, N * 8, cudaMemcpyDeviceToHost);
    for (int i = 8; i < 12; ++i) all.push_back(h[i]);
  }
  // a second executable instantiated from the same graph
  cudaGraphExec_t ge2;
  cudaGraphInstantiate(&ge2, g, 0);
  cudaGraphLaunch(ge2, s2);
  cudaDeviceSynchronize();
  cudaMemcpy(h.data(), d, N * 8, cudaMemcpyDeviceToHost);
  printf("second exec:");
  for (int i = 8; i < 12; ++i) printf(" %llu", h[i]);
  printf("\n");
  std::set<unsigned long long> u(all.begin(), all.end());
  printf("gridids:");
  for (auto v : all) printf(" %llu", v);
  printf("\nlaunches %zu distinct %zu -> %s\n", all.size(), u.size(), all.size() == u.size() ? "UNIQUE" : "DUPLICATES");
  printf("err %s\n", cudaGetErrorString(cudaGetLastError()));
  return 0;
}
