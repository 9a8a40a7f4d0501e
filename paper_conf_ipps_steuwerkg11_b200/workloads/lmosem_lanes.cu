// LM OSEM error-image customizing function for a lanes Map (skel_map_lanes),
// appended to lmosem_error.cu.  Listing 3's loop body for one
// line of response, shared by the `lanes` threads of its group: thread `lane`
// walks piece `lane` of `lanes` equal alpha sub-ranges of the clipped segment
// (walk_piece), the partial forward projections are summed over the group
// (skel_group_sum, so every piece divides by the same fp), and each thread
// back-projects its own piece.  Same image as lmosem_error up to the order of
// float additions (a voxel cut by a piece boundary gets two reductions whose
// lengths add up to its segment length).  Used where one GPU's part of a subset
// is too small to fill the GPU with one thread per event.
void lmosem_lanes(Event e, int lane, int lanes, const float *f, float *c, int nx, int ny, int nz) {
    Walk w;
    const bool ok = walk_piece(e, nx, ny, nz, lane, lanes, w);
    float part = 0.0f;
    if (ok) part = (LMOSEM_VEC_FWD && vec_ok(f, w.nvox)) ? forward_vec(w, f) : forward(w, f);
    const float fp = skel_group_sum(part, lanes);  // every lane of the group calls it
    if (!ok || !(fp > 0.0f)) return;               // empty piece, or empty path (reading R10(iii))
    back_project(w, c, 1.0f / fp);
}
