#!/bin/bash
for defs in "$@"; do echo "== $defs"; SKEL_NVRTC_DEFINES="$defs" python tools/lmosem_scaling_proxy.py; done
