// Probe: can this box create a multicast object (cuMulticastCreate) for the local GPU(s)?
#include <cuda.h>
#include <cstdio>
int main() {
    cuInit(0);
    int ndev = 0;
    cuDeviceGetCount(&ndev);
    CUdevice dev;
    cuDeviceGet(&dev, 0);
    CUcontext ctx;
    cuDevicePrimaryCtxRetain(&ctx, dev);
    cuCtxSetCurrent(ctx);
    int mc = 0, fab = 0, fd = 0;
    cuDeviceGetAttribute(&mc, CU_DEVICE_ATTRIBUTE_MULTICAST_SUPPORTED, dev);
    cuDeviceGetAttribute(&fab, CU_DEVICE_ATTRIBUTE_HANDLE_TYPE_FABRIC_SUPPORTED, dev);
    cuDeviceGetAttribute(&fd, CU_DEVICE_ATTRIBUTE_HANDLE_TYPE_POSIX_FILE_DESCRIPTOR_SUPPORTED, dev);
    printf("devices %d multicast %d fabric %d posix_fd %d\n", ndev, mc, fab, fd);
    for (unsigned nd : {1u, 2u}) {
        for (int ht : {0, 1, 8}) {
            CUmulticastObjectProp p = {};
            p.numDevices = nd;
            p.handleTypes = (CUmemAllocationHandleType)ht;
            p.size = 2u << 20;
            size_t g = 0;
            CUresult rg = cuMulticastGetGranularity(&g, &p, CU_MULTICAST_GRANULARITY_MINIMUM);
            size_t gr = 0;
            cuMulticastGetGranularity(&gr, &p, CU_MULTICAST_GRANULARITY_RECOMMENDED);
            if (g) p.size = ((p.size + g - 1) / g) * g;
            CUmemGenericAllocationHandle h;
            CUresult r = cuMulticastCreate(&h, &p);
            const char *s = nullptr;
            cuGetErrorString(r, &s);
            printf("numDevices %u handleType %d gran %zu (rc %d) rec %zu size %zu -> %d %s\n", nd, ht, g, (int)rg, gr,
                   (size_t)p.size, (int)r, s ? s : "");
            if (r == CUDA_SUCCESS) {
                CUresult ra = cuMulticastAddDevice(h, dev);
                printf("   add device -> %d\n", (int)ra);
                cuMemRelease(h);
            }
        }
    }
    return 0;
}
