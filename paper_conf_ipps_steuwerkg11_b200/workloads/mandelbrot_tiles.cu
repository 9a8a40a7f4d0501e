
// ---- 2-D tiles per warp, appended to mandelbrot_blocked.cu
// A void index Map over the image in tile order: the 32 threads of a warp take
// an 8 x 4 pixel tile instead of 32 pixels of one row, so the lanes' escape
// counts are closer (the warp runs as long as its slowest lane: on the paper's
// image 91.8% of the lane-iterations are useful row by row, 94.7% in 8 x 4
// tiles).  Tile t of the tile-row-major order covers rows 4*(t / (W/8)) ..+3
// and columns 8*(t mod (W/8)) ..+7; each thread writes its count into the
// row-major image `img` (a vector argument).  c is computed exactly as the
// position vector of the plain Map (reading R5).  Needs W % 8 == 0, H % 4 == 0.
void mandelbrot_tiles(unsigned i, int *img, int width, int height, int cap) {
    const unsigned tw = (unsigned)width / 8u;
    const unsigned t = i >> 5, l = i & 31u;
    const unsigned px = (t % tw) * 8u + (l & 7u), py = (t / tw) * 4u + (l >> 3);
    Pos c;
    c.re = (float)(-2.5 + (double)px * (4.0 / (double)width));
    c.im = (float)(-1.5 + (double)py * (3.0 / (double)height));
    img[(unsigned long long)py * (unsigned)width + px] = mandelbrot_blocked(c, cap);
}
