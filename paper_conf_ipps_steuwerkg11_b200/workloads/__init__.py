"""Customizing functions (user source text) of the paper's workloads and of
the skeleton benchmarks.  They are *inputs* to the skeletons, handed to
libskel as strings and compiled by NVRTC into the skeleton
kernels."""
from pathlib import Path

_HERE = Path(__file__).resolve().parent


def source(name: str) -> str:
    return (_HERE / f"{name}.cu").read_text()


MANDELBROT = source("mandelbrot")
LMOSEM_ERROR = source("lmosem_error")
LMOSEM_UPDATE = source("lmosem_update")

# Listing 1, verbatim
SUM_F32 = "float sum (float x,float y){return x+y;}"
MULT_F32 = "float mult(float x,float y){return x*y;}"
SUM_I32 = "int sum(int x, int y){ return x + y; }"
# skeleton sweep
SAXPY_F32 = "float saxpy(float x, float y, float a){ return a * x + y; }"
SAXPY_I32 = "int saxpy(int x, int y, int a){ return a * x + y; }"
MAP_F32 = "float affine(float x){ return x * 2.0f + 1.0f; }"
MAP_I32 = "int affine(int x){ return x * 2 + 1; }"
