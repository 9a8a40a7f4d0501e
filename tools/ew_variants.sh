#!/bin/bash
# element-wise (Map/Zip) tuning sweep: "<SKEL_NVRTC_DEFINES>|<SKEL_EW_WAVES>" per argument
for spec in "$@"; do
  defs="${spec%%|*}"; waves="${spec##*|}"
  SKEL_NVRTC_DEFINES="$defs" SKEL_EW_WAVES="$waves" timeout 200 python bench.py --no-cpu --no-extras --e2e-steps 0 --steps 10 > /tmp/b.json 2>/tmp/b.err
  python -c "
import json; d=json.load(open('/tmp/b.json')); p=d['per_skeleton']; print(repr('$spec'), 'map', round(p['map']['ms'],4), 'zip', round(p['zip']['ms'],4))" || tail -2 /tmp/b.err
done
