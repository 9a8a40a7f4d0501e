// two processes on device 0: A exports a cudaMalloc'd buffer, B opens it (flag from argv)
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <unistd.h>
#include <cuda_runtime.h>
int main(int argc, char** argv) {
  const char* path = "/tmp/ipc_probe.bin";
  cudaSetDevice(0);
  if (argv[1][0] == 'A') {
    void* p; cudaMalloc(&p, 1 << 20); cudaMemset(p, 7, 1 << 20);
    cudaIpcMemHandle_t h; cudaError_t e = cudaIpcGetMemHandle(&h, p);
    printf("A get: %s\n", cudaGetErrorString(e));
    FILE* f = fopen(path, "wb"); fwrite(&h, sizeof h, 1, f); fclose(f);
    sleep(5);
  } else {
    sleep(2);
    cudaIpcMemHandle_t h; FILE* f = fopen(path, "rb"); fread(&h, sizeof h, 1, f); fclose(f);
    void* q = nullptr; unsigned flag = atoi(argv[2]);
    cudaError_t e = cudaIpcOpenMemHandle(&q, h, flag);
    printf("B open flag %u: %s\n", flag, cudaGetErrorString(e));
    if (e == cudaSuccess) { unsigned char c; cudaMemcpy(&c, q, 1, cudaMemcpyDeviceToHost); printf("B read %d\n", c); }
  }
  return 0;
}
