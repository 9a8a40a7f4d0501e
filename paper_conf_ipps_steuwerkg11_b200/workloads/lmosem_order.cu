// On-device event ordering for LM OSEM, built from the
// library's own skeletons: a void Map counts the events of each path-length
// bucket (lm_order_hist), a Scan turns the counts into bucket offsets, and a
// second void Map moves every event into its bucket (lm_order_scatter) --
// longest paths first, so the 32 rays of a warp have similar lengths and the
// longest start first.  List-mode events carry no order and the error image is
// a sum over events (reading R10(x)), so the reordered subset gives the same
// image up to float rounding.  Appended to lmosem_error.cu (walk_clip).
//
// Key: the L1 length |dx|+|dy|+|dz| of the segment clipped to the volume, in
// voxel units -- the number of voxel steps of the walk up to a factor; at
// most nx+ny+nz.  Bucket 0 holds the longest paths.
static __forceinline__ int lm_bucket(const Event &e, int nx, int ny, int nz, int nb) {
    double amin, amax;
    if (!walk_clip(e, nx, ny, nz, amin, amax)) return nb - 1;  // misses the volume: no work, last
    const double l1 = (amax - amin) * (fabs((double)e.x2 - (double)e.x1) + fabs((double)e.y2 - (double)e.y1) +
                                       fabs((double)e.z2 - (double)e.z1));
    const int k = (int)(l1 * (double)nb / (double)(nx + ny + nz));
    return nb - 1 - min(max(k, 0), nb - 1);
}
