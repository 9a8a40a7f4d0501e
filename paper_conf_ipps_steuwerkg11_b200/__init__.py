"""paper_conf_ipps_steuwerkg11_b200 -- SkelCL's data-parallel skeleton hot path
(Steuwer, Kegel, Gorlatch, IPDPS 2011) rebuilt for NVIDIA B200 (sm_100a).

The product is libskel.so (C-ABI in include/skel.h): Vector coherence,
distributions, NVRTC-injected Map/Zip/Reduce/Scan kernels, NCCL exchanges.
`skel` is its ctypes binding; `lmosem` and `workloads` hold the paper's
case studies.
"""
from . import skel  # noqa: F401
from .skel import (BLOCK, COMBINE_ADD, COMBINE_NONE, COPY, SINGLE, Context,  # noqa: F401
                   SkelError, Vector)
