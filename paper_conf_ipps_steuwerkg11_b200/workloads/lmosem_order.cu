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

// Counter slot of an event: bucket-major, LM_ORDER_R replica counters per
// bucket picked by a hash of the event's bits.  With one counter per bucket
// the few busiest buckets serialise ~10^4 atomics each on one L2 address (the
// ordering measured 133 us for 10^6 events); the replicas spread them.  The
// slot depends only on the event, so the counting and the scattering Map
// agree on it, and the scan over the slots in index order still puts the
// buckets in order.
// Each counter sits alone in a 32-byte sector (LM_ORDER_PAD ints apart; the
// zeros between them do not change the scan): atomics on one L2 line are
// serialised, and with consecutive counters the replicas of a busy bucket
// shared four lines.
#define LM_ORDER_R 128
#define LM_ORDER_PAD 8
static __forceinline__ int lm_slot(const Event &e, int nx, int ny, int nz, int nb) {
    unsigned h = __float_as_uint(e.x1) * 0x9E3779B1u ^ __float_as_uint(e.y2) * 0x85EBCA77u ^
                 __float_as_uint(e.z1) * 0xC2B2AE3Du;
    h ^= h >> 15;
    return (lm_bucket(e, nx, ny, nz, nb) * LM_ORDER_R + (int)(h & (LM_ORDER_R - 1))) * LM_ORDER_PAD;
}
