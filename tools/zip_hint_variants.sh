cd "${GRAFT_REPO_ROOT:-/root/repo}"
export PROBE_OPS=zip
echo base; timeout 300 python tools/small_n_probe.py 20 22 30 | cut -c1-90
echo nc_default_st; SKEL_NVRTC_DEFINES='-DSKEL_LD_HINT=".nc" -DSKEL_ST_HINT=""' timeout 300 python tools/small_n_probe.py 20 22 30 | cut -c1-90
echo plain; SKEL_NVRTC_DEFINES='-DSKEL_LD_HINT="" -DSKEL_ST_HINT=""' timeout 300 python tools/small_n_probe.py 20 22 30 | cut -c1-90
