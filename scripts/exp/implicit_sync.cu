// Which host-side CUDA calls serialize a kernel launched AFTER them behind a kernel launched
// BEFORE them on another stream of the same device (the hazard of N logical ranks on one GPU)?
// Stream A: a kernel spinning until stream B's kernel sets a flag (2 s timeout). Between the two
// launches the host makes call X. "blocks" = the spin timed out (B's kernel could not run).
#include <chrono>
#include <cstdio>
#include <cuda_runtime.h>

__global__ void spin(volatile int *flag, int *timed_out) {
    unsigned long long t0, t;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t0));
    while (*flag == 0) {
        asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
        if (t - t0 > 2000000000ull) { *timed_out = 1; return; }
    }
}
__global__ void setflag(int *flag) { *flag = 1; }
__global__ void fresh_kernel(int *x) { *x += 1; }  // first launch happens in the test (lazy load)

int main() {
    cudaStream_t a, b;
    cudaStreamCreateWithFlags(&a, cudaStreamNonBlocking);
    cudaStreamCreateWithFlags(&b, cudaStreamNonBlocking);
    int *flag, *to, *scratch;
    cudaMalloc(&flag, 4); cudaMalloc(&to, 4); cudaMalloc(&scratch, 4);
    const char *names[] = {"none", "cudaMalloc", "cudaMallocAsync", "cudaMallocHost", "cudaHostAlloc",
                           "cudaFree", "cudaFreeAsync", "cudaMemset", "cudaMemsetAsync", "cudaEventCreate",
                           "lazy first launch", "cudaFreeHost", "cudaMemcpy D2H", "cudaHostRegister"};
    for (int x = 0; x < 14; ++x) {
        cudaMemset(flag, 0, 4); cudaMemset(to, 0, 4); cudaDeviceSynchronize();
        void *p = nullptr, *q = nullptr;
        if (x == 5) cudaMalloc(&q, 1 << 20);
        if (x == 6) cudaMallocAsync(&q, 1 << 20, b);
        if (x == 11) cudaMallocHost(&q, 1 << 20);
        static char hostbuf[1 << 16];
        cudaDeviceSynchronize();
        spin<<<1, 1, 0, a>>>(flag, to);
        auto t0 = std::chrono::steady_clock::now();
        switch (x) {
            case 1: cudaMalloc(&p, 64 << 20); break;
            case 2: cudaMallocAsync(&p, 64 << 20, b); break;
            case 3: cudaMallocHost(&p, 1 << 20); break;
            case 4: cudaHostAlloc(&p, 1 << 20, cudaHostAllocMapped); break;
            case 5: cudaFree(q); break;
            case 6: cudaFreeAsync(q, b); break;
            case 7: cudaMemset(scratch, 0, 4); break;
            case 8: cudaMemsetAsync(scratch, 0, 4, b); break;
            case 9: { cudaEvent_t e; cudaEventCreate(&e); break; }
            case 10: fresh_kernel<<<1, 1, 0, b>>>(scratch); break;
            case 11: cudaFreeHost(q); break;
            case 12: { int h; cudaMemcpy(&h, scratch, 4, cudaMemcpyDeviceToHost); break; }
            case 13: cudaHostRegister(hostbuf, sizeof hostbuf, 0); break;
        }
        const double host_ms = std::chrono::duration<double, std::milli>(std::chrono::steady_clock::now() - t0).count();
        setflag<<<1, 1, 0, b>>>(flag);
        cudaDeviceSynchronize();
        int timed = 0;
        cudaMemcpy(&timed, to, 4, cudaMemcpyDeviceToHost);
        printf("%-20s host call %8.2f ms  -> %s\n", names[x], host_ms, timed ? "BLOCKS (serialised behind the spinner)" : "ok");
        if (x == 1 || x == 5) cudaFree(p);
        if (x == 2) cudaFreeAsync(p, b);
        if (x == 3 || x == 4) cudaFreeHost(p);
        if (x == 13) cudaHostUnregister(hostbuf);
        cudaDeviceSynchronize();
    }
    printf("err: %s\n", cudaGetErrorString(cudaGetLastError()));
    return 0;
}
