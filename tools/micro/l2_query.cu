#include <cstdio>
#include <cuda_runtime.h>
int main(){int v; cudaDeviceGetAttribute(&v, cudaDevAttrMaxPersistingL2CacheSize, 0); printf("max persisting L2 %d\n", v);
cudaDeviceGetAttribute(&v, cudaDevAttrMaxAccessPolicyWindowSize, 0); printf("max window %d\n", v);
cudaDeviceGetAttribute(&v, cudaDevAttrL2CacheSize, 0); printf("L2 %d\n", v);
cudaDeviceGetAttribute(&v, cudaDevAttrCooperativeLaunch, 0); printf("coop %d\n", v); return 0;}
