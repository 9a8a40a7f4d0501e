#!/bin/bash
# scan tuning sweep: prints scan ms and fraction of measured HBM per -D set
for defs in "$@"; do
  SKEL_NVRTC_DEFINES="$defs" timeout 200 python bench.py --no-cpu --no-extras --e2e-steps 0 --steps 10 > /tmp/b.json 2>/tmp/b.err
  python -c "
import json,sys; d=json.load(open('/tmp/b.json')); print(repr('$defs'), round(d['per_skeleton']['scan']['ms'],3), round(d['per_skeleton']['scan']['frac_of_hbm'],3))" || tail -2 /tmp/b.err
done
