import os, sys
sys.path.insert(0, os.getcwd())
import numpy as np, torch
from paper_conf_ipps_steuwerkg11_b200 import skel
H = r'''
static __forceinline__ unsigned ph(unsigned x){ x^=x>>16; x*=0x7feb352du; x^=x>>15; x*=0x846ca68bu; x^=x>>16; return x; }
'''
SRC = {
 "red1": H + r'''void p(unsigned i, float* c, unsigned n){ for(int k=0;k<64;++k){ float* q=&c[ph(i*64+k)%n]; asm volatile("red.global.add.f32 [%0], %1;"::"l"(q),"f"(1.0f):"memory"); } }''',
 "red2": H + r'''void p(unsigned i, float* c, unsigned n){ for(int k=0;k<64;++k){ float* q=&c[(ph(i*64+k)%n)&~1u]; asm volatile("red.global.add.v2.f32 [%0], {%1,%2};"::"l"(q),"f"(1.0f),"f"(1.0f):"memory"); } }''',
 "red4": H + r'''void p(unsigned i, float* c, unsigned n){ for(int k=0;k<64;++k){ float* q=&c[(ph(i*64+k)%n)&~3u]; asm volatile("red.global.add.v4.f32 [%0], {%1,%2,%3,%4};"::"l"(q),"f"(1.0f),"f"(1.0f),"f"(1.0f),"f"(1.0f):"memory"); } }''',
}
with skel.Context(1) as ctx:
    st = torch.cuda.ExternalStream(ctx.stream(0))
    N = 1 << 20
    idx = ctx.vector(np.arange(N, dtype=np.uint32))
    c = ctx.vector(n=150*150*280, dtype=np.float32).fill(np.float32(0))
    for name, src in SRC.items():
        for n in (150*150*280, 1 << 18):
            a = [c, np.uint32(n)]
            for _ in range(2): ctx.map(src, idx, None, args=a)
            ctx.sync()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(st)
            for _ in range(10): ctx.map(src, idx, None, args=a)
            e1.record(st); ctx.sync()
            ms = e0.elapsed_time(e1) / 10
            print(name, n, f"{ms:.3f} ms", f"{N*64/ms/1e6:.1f} G instr-req/s")
